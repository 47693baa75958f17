"""Pins for the oracle's arithmetic (oracle/chol_oracle.c) against things other than
itself: LAPACK (numpy/scipy), exact integer factors, closed forms, special cases
that reduce to textbook routines, and the non-SPD convention.  CPU only."""
import numpy as np
import pytest
import scipy.linalg as sla

import oracle
import spdgen


def lapack_chol(A):
    return np.linalg.cholesky(np.tril(A) + np.tril(A, -1).T)


@pytest.mark.parametrize("n", [1, 2, 3, 7, 64, 200])
def test_unblocked_matches_lapack(n):
    A = spdgen.uniform_spd(n, seed=n)
    L, info = oracle.chol_unblocked(A)
    assert info == 0
    d = oracle.rel_diff(L, lapack_chol(A))
    assert d["max_rel_floored"] < 1e-13, d


@pytest.mark.parametrize("n,nb", [(64, 16), (96, 32), (250, 50), (256, 64), (1024, 256)])
def test_tiled_matches_lapack(n, nb):
    A = spdgen.uniform_spd(n, seed=3)
    L, info = oracle.chol_tiled(A, nb)
    assert info == 0
    d = oracle.rel_diff(L, lapack_chol(A))
    assert d["max_rel_floored"] < 1e-12, d
    assert np.all(np.triu(L, 1) == 0.0)
    assert np.all(np.diag(L) > 0)


@pytest.mark.parametrize("n,nb,seed", [(64, 16, 0), (96, 32, 1), (256, 64, 2), (1024, 256, 5),
                                       (120, 8, 7)])
def test_integer_family_exact(n, nb, seed):
    """A = L0 L0^T with integer L0 (reading R16 / SURVEY §8c): any correct
    algorithm returns exactly L0, bit for bit."""
    L0 = spdgen.integer_L0(n, seed)
    A = spdgen.integer_spd(n, seed)
    assert np.array_equal(A, L0 @ L0.T)  # the generator's banded product is right
    L, info = oracle.chol_tiled(A, nb)
    assert info == 0 and np.array_equal(L, L0)
    Lu, info = oracle.chol_unblocked(A)
    assert info == 0 and np.array_equal(Lu, L0)


def test_known_floating_factor():
    rng = np.random.default_rng(11)
    n = 300
    L0 = np.tril(rng.uniform(-1, 1, (n, n)), -1) / np.sqrt(n) + np.diag(rng.uniform(1, 2, n))
    A = L0 @ L0.T
    L, info = oracle.chol_tiled(A, 60)
    assert info == 0
    kappa = np.linalg.cond(A)
    err = np.linalg.norm(L - L0) / np.linalg.norm(L0)
    assert err < 50 * kappa * np.finfo(float).eps, (err, kappa)


def test_single_tile_is_unblocked():
    """N = 1 (nb = n): Algorithm 1 is a single POTRF."""
    A = spdgen.uniform_spd(97, seed=2)
    assert np.array_equal(oracle.chol_tiled(A, 97)[0], oracle.chol_unblocked(A)[0])


def test_nb_one_is_outer_product_cholesky():
    """nb = 1: Algorithm 1 degenerates to the scalar right-looking (outer product)
    Cholesky; compare with LAPACK."""
    A = spdgen.uniform_spd(40, seed=4)
    L, info = oracle.chol_tiled(A, 1)
    assert info == 0
    assert oracle.rel_diff(L, lapack_chol(A))["max_rel_floored"] < 1e-13


def test_two_by_two_tiles_closed_form():
    """N = 2: L00 = chol(A00), L10 = A10 L00^-T, L11 = chol(A11 - L10 L10^T),
    each step computed by LAPACK / scipy."""
    n, nb = 128, 64
    A = spdgen.uniform_spd(n, seed=9)
    A00, A10, A11 = A[:nb, :nb], A[nb:, :nb], A[nb:, nb:]
    L00 = np.linalg.cholesky(np.tril(A00) + np.tril(A00, -1).T)
    L10 = sla.solve_triangular(L00, A10.T, lower=True).T
    S = A11 - L10 @ L10.T
    L11 = np.linalg.cholesky(np.tril(S) + np.tril(S, -1).T)
    ref = np.zeros_like(A)
    ref[:nb, :nb], ref[nb:, :nb], ref[nb:, nb:] = L00, L10, L11
    L, info = oracle.chol_tiled(A, nb)
    assert info == 0
    assert oracle.rel_diff(L, ref)["max_rel_floored"] < 1e-13


def test_reads_lower_triangle_only():
    n, nb = 192, 64
    A = spdgen.uniform_spd(n, seed=1)
    An = spdgen.uniform_spd(n, seed=1, upper="nan")
    assert np.array_equal(oracle.chol_tiled(A, nb)[0], oracle.chol_tiled(An, nb)[0])
    Ai = spdgen.integer_spd(n, 1, upper="nan")
    assert np.array_equal(oracle.chol_tiled(Ai, nb)[0], spdgen.integer_L0(n, 1))


@pytest.mark.parametrize("kind", ["zero", "neg"])
@pytest.mark.parametrize("j0", [0, 64, 64 + 37, 255])
def test_non_spd_info(j0, kind):
    """info = j0 + 1 (1-based column of the first non-positive pivot, reading R6)."""
    n, nb = 256, 64
    L0 = spdgen.integer_L0(n, 3)
    A = spdgen.make_non_spd(spdgen.integer_spd(n, 3), L0, j0, kind)
    assert oracle.chol_tiled(A, nb)[1] == j0 + 1
    assert oracle.chol_unblocked(A)[1] == j0 + 1


def test_nan_pivot_is_rejected():
    A = spdgen.uniform_spd(64, seed=0)
    A[40, 40] = np.nan
    assert oracle.chol_tiled(A, 16)[1] == 41


def test_backward_error_within_north_star():
    n = 1024
    A = spdgen.uniform_spd(n, seed=0)
    L, info = oracle.chol_tiled(A, 256)
    assert info == 0
    assert oracle.backward_error(A, L) <= 10.0


def test_tile_ops_match_library():
    rng = np.random.default_rng(5)
    nb = 48
    M = rng.standard_normal((nb, nb))
    S = M @ M.T + nb * np.eye(nb)
    Lkk, info = oracle.tile_potrf(S)
    assert info == 0
    assert np.allclose(np.tril(Lkk), np.linalg.cholesky(S), rtol=1e-13, atol=1e-13)
    Lkk = np.tril(Lkk)
    B = rng.standard_normal((nb, nb))
    X = oracle.tile_trsm(Lkk, B)
    assert np.allclose(X, sla.solve_triangular(Lkk, B.T, lower=True).T, rtol=1e-12, atol=1e-12)
    assert np.allclose(X @ Lkk.T, B, rtol=1e-12, atol=1e-12)
    A1, A2, C = (rng.standard_normal((nb, nb)) for _ in range(3))
    G = oracle.tile_gemm(A1, A2, C)
    assert np.allclose(G, C - A1 @ A2.T, rtol=1e-13, atol=1e-12)
    Y = oracle.tile_syrk(A1, C)
    tri = np.tril_indices(nb)
    assert np.allclose(Y[tri], (C - A1 @ A1.T)[tri], rtol=1e-13, atol=1e-12)
    assert np.array_equal(np.triu(Y, 1), np.triu(C, 1))  # upper untouched


def test_flop_count_identity():
    """Per-kernel LAPACK counts nb^3/3+nb^2/2+nb/6 (POTRF), nb^3 (TRSM), nb^2(nb+1)
    (SYRK), 2nb^3 (GEMM) times the task counts sum to n^3/3+n^2/2+n/6 (reading R7)."""
    from oracle import bounds
    from fractions import Fraction as F
    for N in range(1, 30):
        for nb in (1, 2, 7, 960):
            c = bounds.task_counts(N)
            tot = (c["POTRF"] * (F(nb ** 3, 3) + F(nb ** 2, 2) + F(nb, 6)) + c["TRSM"] * nb ** 3
                   + c["SYRK"] * nb ** 2 * (nb + 1) + c["GEMM"] * 2 * nb ** 3)
            n = N * nb
            assert tot == F(n ** 3, 3) + F(n ** 2, 2) + F(n, 6)
