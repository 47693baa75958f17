"""The shared seeded input generator (spdgen) -- structure checks."""
import numpy as np

import spdgen


def test_uniform_symmetric_and_spd():
    A = spdgen.uniform_spd(300, seed=5)
    assert np.array_equal(A, A.T)
    off = np.abs(A - np.diag(np.diag(A))).sum(1)
    assert np.all(np.diag(A) - off > 0)  # Gershgorin: strictly diagonally dominant
    assert A.min() >= -0.5 and np.max(np.abs(A - np.diag(np.diag(A)))) < 0.5


def test_uniform_row_slices_match():
    A = spdgen.uniform_spd(100, seed=2)
    B = spdgen.uniform_spd(100, seed=2, rows=slice(30, 70))
    assert np.array_equal(A[30:70], B)


def test_splitmix64_reference_values():
    # splitmix64 stream from seed 0 (state advanced by the golden gamma each call):
    # first outputs 0xE220A8397B1DCDAF, 0x6E789E6AA1B965F4 (Vigna's reference generator)
    z = spdgen.splitmix64(np.array([0, 0x9E3779B97F4A7C15], dtype=np.uint64))
    assert int(z[0]) == 0xE220A8397B1DCDAF
    assert int(z[1]) == 0x6E789E6AA1B965F4


def test_integer_family_structure():
    L0 = spdgen.integer_L0(200, 3)
    assert set(np.unique(np.diag(L0))) <= {1.0, 2.0, 4.0}
    off = L0[np.tril_indices(200, -1)]
    assert set(np.unique(off)) <= {-1.0, 0.0, 1.0}
    assert np.all(np.triu(L0, 1) == 0)
    assert np.all(np.tril(L0, -spdgen.BW - 1) == 0)
    A = spdgen.integer_spd(200, 3)
    assert np.array_equal(A, L0 @ L0.T)


def test_uniform_entries_match_dense():
    n = 77
    A = spdgen.uniform_spd(n, seed=3)
    rng = np.random.default_rng(0)
    i = rng.integers(0, n, 500)
    j = rng.integers(0, n, 500)
    assert np.array_equal(spdgen.uniform_entries(n, 3, i, j), A[i, j])


def test_integer_family_block_inverses_are_exact():
    """DESIGN R19: the inverse-form TRSM keeps the integer family exact because the inverses
    of L0's diagonal 96-blocks (and whole 960-tiles) are small dyadic numbers.  Checked in
    exact rational arithmetic on a few blocks (forward substitution with Fractions: every entry
    is dyadic with a numerator below 2^53, i.e. exactly representable in FP64), and in FP64 on
    every 96-block: the FP64 inverse times the block is the identity exactly."""
    from fractions import Fraction
    import numpy as np
    for seed in (0, 3, 12):
        n = 3840
        L0 = spdgen.integer_L0(n, seed)
        for b in range(0, n, 96):
            L = L0[b:b + 96, b:b + 96]
            X = np.linalg.solve(L, np.eye(96))
            assert np.array_equal(L @ X, np.eye(96))
            assert np.abs(X).max() <= 64.0
        for b in (0, 960, 2880):  # exact rationals: every entry dyadic with a small numerator
            L = [[Fraction(int(v)) for v in row] for row in L0[b:b + 96, b:b + 96]]
            for col in range(96):
                x = [Fraction(0)] * 96
                for r in range(96):
                    s = Fraction(1 if r == col else 0) - sum(L[r][m] * x[m] for m in range(max(0, r - 3), r))
                    x[r] = s / L[r][r]
                for v in x:
                    assert v.denominator & (v.denominator - 1) == 0  # power of two
                    assert abs(v.numerator) < 2 ** 53  # exactly representable in FP64
                    assert Fraction(float(v)) == v
