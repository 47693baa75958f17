"""chol_solve on the GPU against the oracle's substitution with the
same factor: several tile / block sizes, ragged right-hand-side counts (1, 5, 32, 33, 70
-> padded 32-column chunks), host and device B, ldb > nrhs, the full bench size, and the
error paths (no factor, failed factor, bad arguments).

Tolerance: the library applies each bs x bs diagonal block through its
explicit inverse, the oracle substitutes; for the well-conditioned uniform family
(kappa <~ 3) both are within a few n eps of X, so max|X - X^| <= 1e-12 max|X^|, and the
residual ||A X - B|| / (||A|| ||X|| n eps) <= 10."""
import numpy as np
import pytest

import oracle
import spdgen

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")


def _lib():
    import paper_conf_ipps_agullobehkmt15_b200 as c
    return c


def _factor(c, n, nb, seed=0, **opts):
    A = spdgen.uniform_spd(n, seed)
    p = c.Plan(n, nb, **opts)
    dA = torch.from_numpy(A).cuda()
    assert p.factor(dA) == 0
    torch.cuda.synchronize()
    return p, A, dA.cpu().numpy()


def _check(A, L, B, X):
    ref = oracle.chol_solve(L, B)
    scale = max(1.0, float(np.max(np.abs(ref))))
    assert np.max(np.abs(X - ref)) <= 1e-12 * scale
    n = A.shape[0]
    r = np.linalg.norm(A @ X - B) / (np.linalg.norm(A) * np.linalg.norm(X) * n * np.finfo(np.float64).eps)
    assert r <= 10.0, r


@pytest.mark.parametrize("n,nb", [(1024, 256), (3840, 960), (1920, 96), (768, 64), (2880, 960), (640, 32)])
@pytest.mark.parametrize("nrhs", [1, 5, 33])
def test_solve_matches_oracle(n, nb, nrhs):
    c = _lib()
    p, A, L = _factor(c, n, nb)
    with p:
        B = spdgen.rhs(n, nrhs, 7)
        X = B.copy()
        p.solve(X)  # host pointer
        _check(A, L, B, X)
        dB = torch.from_numpy(B).cuda()  # device pointer, same answer bit for bit
        p.solve(dB)
        torch.cuda.synchronize()
        assert np.array_equal(dB.cpu().numpy(), X)


@pytest.mark.parametrize("nrhs", [1, 32, 70])
def test_solve_padded_ldb_and_repeat(nrhs):
    c = _lib()
    n, nb = 1920, 960
    p, A, L = _factor(c, n, nb, seed=3)
    with p:
        ldb = nrhs + 9
        Bw = np.full((n, ldb), 123.0)
        B = spdgen.rhs(n, nrhs, 1)
        Bw[:, :nrhs] = B
        c.chol_solve(p.h, Bw, ldb, nrhs)
        _check(A, L, B, Bw[:, :nrhs].copy())
        assert np.all(Bw[:, nrhs:] == 123.0)  # columns beyond nrhs untouched
        X2 = B.copy()
        p.solve(X2)  # second solve reuses the diagonal-block inverses
        assert np.array_equal(X2, Bw[:, :nrhs])


def test_solve_after_refactor_uses_new_factor():
    c = _lib()
    n, nb = 1920, 960
    with c.Plan(n, nb) as p:
        A1 = spdgen.uniform_spd(n, 1)
        A2 = spdgen.uniform_spd(n, 2)
        B = spdgen.rhs(n, 3, 0)
        for A in (A1, A2):
            dA = torch.from_numpy(A).cuda()
            assert p.factor(dA) == 0
            torch.cuda.synchronize()
            X = B.copy()
            p.solve(X)
            _check(A, dA.cpu().numpy(), B, X)


def test_solve_full_size():
    """The bench size n = 19200 (nb = 960), one right-hand side and a 32-column chunk."""
    c = _lib()
    n, nb = 19200, 960
    with c.Plan(n, nb) as p:
        c.chol_generate(p.h, 0, 0)
        assert c.chol_factor_inplace(p.h) == 0
        L = np.zeros((n, n))
        c.chol_gather(p.h, L, n)
        A = spdgen.uniform_spd(n, 0)
        for nrhs in (1, 32):
            B = spdgen.rhs(n, nrhs, 5)
            X = B.copy()
            p.solve(X)
            _check(A, L, B, X)


def test_solve_errors():
    c = _lib()
    n, nb = 1024, 256
    with c.Plan(n, nb) as p:
        B = spdgen.rhs(n, 2, 0)
        with pytest.raises(c.CholError) as e:
            p.solve(B)  # nothing factored yet
        assert e.value.status == -10
        L0 = spdgen.integer_L0(n, 3)
        Abad = spdgen.make_non_spd(spdgen.integer_spd(n, 3), L0, 300, "zero")
        dA = torch.from_numpy(Abad).cuda()
        assert p.factor(dA) == 301
        with pytest.raises(c.CholError) as e:
            p.solve(B)  # the last factorization failed
        assert e.value.status == -10
        dA = torch.from_numpy(spdgen.uniform_spd(n, 0)).cuda()
        assert p.factor(dA) == 0
        with pytest.raises(c.CholError) as e:
            c.chol_solve(p.h, B, 1, 2)
        assert e.value.status == -5
        with pytest.raises(c.CholError) as e:
            c.chol_solve(p.h, B, 2, 0)
        assert e.value.status == -6


@pytest.mark.parametrize("nrhs", [2, 8, 40])
def test_solve_dmma_and_simt_sweeps_agree(nrhs, monkeypatch):
    """Block 96 runs the DMMA sweeps (k_sweep_mma); CHOL_SOLVE_SIMT=1 the SIMT ones
    (k_sweep): both against the oracle, and against each other within the same bound."""
    c = _lib()
    n, nb = 2880, 960
    p, A, L = _factor(c, n, nb, seed=3)
    B = spdgen.rhs(n, nrhs, 9)
    X1 = B.copy()
    p.solve(X1)
    _check(A, L, B, X1)
    p.close()
    monkeypatch.setenv("CHOL_SOLVE_SIMT", "1")
    p, _, _ = _factor(c, n, nb, seed=3)
    X2 = B.copy()
    p.solve(X2)
    p.close()
    _check(A, L, B, X2)
    assert np.max(np.abs(X1 - X2)) <= 1e-12 * max(1.0, float(np.max(np.abs(X1))))


@pytest.mark.parametrize("rc", ["32", "48", "64"])
@pytest.mark.parametrize("n,nrhs", [(3840, 101), (9600, 49)])
def test_solve_chunk_widths_match_oracle(rc, n, nrhs, monkeypatch):
    """Every chunk width of the block-96 DMMA sweeps -- 32 / 64 (k_sweep_mma) and 48
    (k_sweep_db, both operands double-buffered, swizzled shared layout) -- forced with
    CHOL_SOLVE_RC, ragged last chunk, against the oracle."""
    c = _lib()
    monkeypatch.setenv("CHOL_SOLVE_RC", rc)
    p, A, L = _factor(c, n, 960, seed=4)
    B = spdgen.rhs(n, nrhs, 11)
    X = B.copy()
    p.solve(X)
    p.close()
    _check(A, L, B, X)


def test_solve_refuses_a_factor_that_was_overwritten_or_failed():
    """Every call that writes the tile store (generate, scatter, run_batch / run_task, a
    factorization that fails) invalidates the factor: chol_solve returns -10 instead of
    solving with stale data or stale cached inverses."""
    c = _lib()
    n, nb = 1920, 960
    B = torch.from_numpy(spdgen.rhs(n, 3, 1)).cuda()
    with c.Plan(n, nb) as p:

        def expect_stale():
            with pytest.raises(c.CholError) as e:
                p.solve(B.clone())
            assert e.value.status == -10

        def refactor():
            c.chol_generate(p.h, 3, 0)
            assert c.chol_factor_inplace(p.h) == 0
            p.solve(B.clone())  # fine again

        refactor()
        c.chol_generate(p.h, 4, 0)
        expect_stale()
        refactor()
        c.chol_scatter(p.h, torch.from_numpy(spdgen.uniform_spd(n, 5)).cuda(), n)
        expect_stale()
        refactor()
        c.chol_run_batch(p.h, c.GEMM if n // nb > 2 else c.SYRK, 1)
        expect_stale()
        refactor()
        L0 = spdgen.integer_L0(n, 2)
        bad = torch.from_numpy(spdgen.make_non_spd(spdgen.integer_spd(n, 2), L0, 1000)).cuda()
        assert p.factor(bad) == 1001
        expect_stale()
