"""GPU parity: the CUDA path (through the C-ABI) against the CPU oracle on the same
seeded inputs (spdgen).  Tolerances: north star -- backward error
||A - L L^T||_F / (n eps ||A||_F) <= 10 and floored max relative elementwise
difference <= 1e-10 (reading R8); bitwise equality on the exact integer family
and for the non-SPD info code."""
import numpy as np
import pytest

import oracle
import spdgen

pytestmark = pytest.mark.gpu

torch = pytest.importorskip("torch")

EXECUTORS = ["host", "sched"]


def _lib():
    import paper_conf_ipps_agullobehkmt15_b200 as c
    return c


def _opts(executor, **kw):
    c = _lib()
    kw.setdefault("executor", c.EXEC_HOST if executor == "host" else c.EXEC_SCHEDULER)
    return kw


def gpu_factor(A: np.ndarray, nb: int, executor="sched", device_ptrs=True, **opts):
    c = _lib()
    n = A.shape[0]
    with c.Plan(n, nb, **_opts(executor, **opts)) as p:
        if device_ptrs:
            dA = torch.from_numpy(np.ascontiguousarray(A)).cuda()
            info = p.factor(dA)
            torch.cuda.synchronize()
            return dA.cpu().numpy(), info
        L = np.empty_like(A)
        info = p.factor(np.ascontiguousarray(A), L)
        return L, info


# ----------------------------------------------------------------------- tile ops
def _scatter_run(n, nb, M, type_, i, j, k):
    c = _lib()
    with c.Plan(n, nb, executor=c.EXEC_HOST) as p:
        dM = torch.from_numpy(np.ascontiguousarray(M)).cuda()
        c.chol_scatter(p.h, dM, n)
        c.chol_run_task(p.h, type_, i, j, k, 1)
        out = torch.empty_like(dM)
        c.chol_gather(p.h, out, n)
        torch.cuda.synchronize()
        return out.cpu().numpy()


def _T(M, nb, i, j):
    return M[i * nb:(i + 1) * nb, j * nb:(j + 1) * nb]


def _close(a, b, tol=1e-10):
    """Floored relative difference (reading R8) at the north-star tolerance."""
    scale = max(np.max(np.abs(b)), 1e-300)
    d = np.abs(a - b) / np.maximum(np.abs(b), 1e-6 * scale)
    assert np.max(d) <= tol, float(np.max(d))


def _gemm_close(got, ref, C, A, B, mask=None):
    """GPU vs oracle for C - A B^T: both are within the componentwise forward-error
    bound 2 K eps (|C| + |A| |B|^T) of the exact result (Higham, Thm 3.5), so
    |got - ref| <= 2 x that bound.  (The relative floor of _close is meaningless
    where the update cancels to ~0.)"""
    K = A.shape[1]
    bound = 2 * K * np.finfo(float).eps * (np.abs(C) + np.abs(A) @ np.abs(B).T)
    err = np.abs(got - ref)
    if mask is not None:
        err, bound = err[mask], bound[mask]
    assert np.all(err <= 2 * bound), float(np.max(err / np.maximum(bound, 1e-300)))


@pytest.mark.parametrize("nb", [96, 64, 160, 256, 960])
def test_tile_potrf(nb):
    c = _lib()
    n = 3 * nb
    M = spdgen.uniform_spd(n, seed=21)
    out = _scatter_run(n, nb, M, c.POTRF, 1, 1, 1)
    ref, info = oracle.tile_potrf(_T(M, nb, 1, 1))
    assert info == 0
    _close(np.tril(_T(out, nb, 1, 1)), np.tril(ref))


@pytest.mark.parametrize("nb", [96, 64, 160, 256, 960])
def test_tile_trsm(nb):
    c = _lib()
    n = 3 * nb
    M = spdgen.uniform_spd(n, seed=22)
    out = _scatter_run(n, nb, M, c.TRSM, 2, 0, 0)
    ref = oracle.tile_trsm(np.tril(_T(M, nb, 0, 0)), _T(M, nb, 2, 0))
    _close(_T(out, nb, 2, 0), ref)


@pytest.mark.parametrize("nb", [96, 64, 160, 256, 960])
def test_tile_syrk(nb):
    c = _lib()
    n = 3 * nb
    M = spdgen.uniform_spd(n, seed=23)
    out = _scatter_run(n, nb, M, c.SYRK, 1, 1, 0)
    A1, C = _T(M, nb, 1, 0), _T(M, nb, 1, 1)
    ref = oracle.tile_syrk(A1, C)
    _gemm_close(_T(out, nb, 1, 1), ref, C, A1, A1, mask=np.tril(np.ones((nb, nb), dtype=bool)))


@pytest.mark.parametrize("nb", [96, 64, 160, 256, 960])
def test_tile_gemm(nb):
    c = _lib()
    n = 3 * nb
    M = spdgen.uniform_spd(n, seed=24)
    out = _scatter_run(n, nb, M, c.GEMM, 2, 1, 0)
    A, B, C = _T(M, nb, 2, 0), _T(M, nb, 1, 0), _T(M, nb, 2, 1)
    _gemm_close(_T(out, nb, 2, 1), oracle.tile_gemm(A, B, C), C, A, B)


# ----------------------------------------------------------------------- whole factorization
CASES = [(1024, 256), (96, 96), (64, 32), (288, 96), (640, 160), (1920, 960), (2880, 960)]


@pytest.mark.parametrize("executor", EXECUTORS)
@pytest.mark.parametrize("n,nb", CASES)
def test_factor_matches_oracle(n, nb, executor):
    A = spdgen.uniform_spd(n, seed=n + nb)
    L, info = gpu_factor(A, nb, executor)
    ref, rinfo = oracle.chol_tiled(A, nb)
    assert info == rinfo == 0
    d = oracle.rel_diff(L, ref)
    assert d["max_rel_floored"] <= 1e-10, d
    assert np.all(np.triu(L, 1) == 0.0)
    assert oracle.backward_error(A, L) <= 10.0


@pytest.mark.parametrize("executor", EXECUTORS)
@pytest.mark.parametrize("n,nb,seed", [(1024, 256, 0), (1920, 960, 1), (576, 96, 2), (640, 160, 3)])
def test_integer_family_bitwise(n, nb, seed, executor):
    A = spdgen.integer_spd(n, seed)
    L, info = gpu_factor(A, nb, executor)
    assert info == 0
    assert np.array_equal(L, spdgen.integer_L0(n, seed))


@pytest.mark.parametrize("executor", EXECUTORS)
@pytest.mark.parametrize("kind", ["zero", "neg"])
@pytest.mark.parametrize("j0", [0, 96 + 37, 2 * 96, 575])
def test_non_spd_info(j0, kind, executor):
    n, nb = 576, 96
    L0 = spdgen.integer_L0(n, 4)
    A = spdgen.make_non_spd(spdgen.integer_spd(n, 4), L0, j0, kind)
    _, info = gpu_factor(A, nb, executor)
    assert info == j0 + 1 == oracle.chol_tiled(A, nb)[1]


@pytest.mark.parametrize("executor", EXECUTORS)
def test_reads_lower_only_and_host_pointers(executor):
    n, nb = 960, 96
    A = spdgen.uniform_spd(n, seed=5)
    An = spdgen.uniform_spd(n, seed=5, upper="nan")
    L1, i1 = gpu_factor(A, nb, executor)
    L2, i2 = gpu_factor(An, nb, executor)
    L3, i3 = gpu_factor(An, nb, executor, device_ptrs=False)
    assert i1 == i2 == i3 == 0
    assert np.array_equal(L1, L2) and np.array_equal(L1, L3)


def test_bitwise_identical_across_executors_and_policies():
    """Reading R15: each tile's update order is fixed by the DAG, so L does not
    depend on the schedule."""
    c = _lib()
    n, nb = 1920, 96
    A = spdgen.uniform_spd(n, seed=8)
    ref, _ = gpu_factor(A, nb, "host")
    for pol in (c.POLICY_DYNAMIC, c.POLICY_CP_PRIORITY, c.POLICY_STATIC):
        L, info = gpu_factor(A, nb, "sched", policy=pol)
        assert info == 0 and np.array_equal(L, ref), pol


@pytest.mark.parametrize("family", [0, 1])
def test_device_generator_matches_spdgen(family):
    c = _lib()
    n, nb = 640, 160
    with c.Plan(n, nb, executor=c.EXEC_HOST) as p:
        c.chol_generate(p.h, 7, family)
        out = torch.empty((n, n), dtype=torch.float64, device="cuda")
        c.chol_gather(p.h, out, n)
        torch.cuda.synchronize()
        got = out.cpu().numpy()
    ref = spdgen.uniform_spd(n, 7) if family == 0 else spdgen.integer_spd(n, 7)
    assert np.array_equal(got, np.tril(ref))


def test_lda_larger_than_n():
    n, nb, lda = 384, 96, 400
    A = spdgen.uniform_spd(n, seed=9)
    Ab = np.full((n, lda), np.nan)
    Ab[:, :n] = A
    c = _lib()
    with c.Plan(n, nb) as p:
        dA = torch.from_numpy(Ab).cuda()
        dL = torch.full((n, lda), 7.0, dtype=torch.float64, device="cuda")
        info = c.chol_factor(p.h, dA, lda, dL, lda)
        L = dL.cpu().numpy()
    assert info == 0
    assert np.all(L[:, n:] == 7.0)  # padding untouched
    ref, _ = oracle.chol_tiled(A, nb)
    assert oracle.rel_diff(L[:, :n], ref)["max_rel_floored"] <= 1e-10


def test_argument_errors():
    c = _lib()
    with pytest.raises(c.CholError) as e:
        c.chol_plan(0, 32)
    assert e.value.status == -1
    for n, nb in [(100, 32), (96, 0), (96, 48)]:
        with pytest.raises(c.CholError) as e:
            c.chol_plan(n, nb)
        assert e.value.status == -2
    with pytest.raises(c.CholError) as e:
        c.chol_plan(96, 32, 999)
    assert e.value.status == -3
    with pytest.raises(c.CholError) as e:
        c.chol_plan_ex(96, 32, 1, policy=7)
    assert e.value.status == -6
    for bad in (dict(cpu_trsm_distance=-1), dict(cpu_threads=-2), dict(cpu_trsm_distance=2, executor=c.EXEC_HOST)):
        with pytest.raises(c.CholError) as e:
            c.chol_plan_ex(960, 96, 1, **bad)
        assert e.value.status == -6
    with pytest.raises(c.CholError) as e:  # the host CPU class is single-GPU only
        c.chol_plan_dist(960, 96, 2, 0, cpu_trsm_distance=2)
    assert e.value.status == -6
    with c.Plan(96, 32) as p:
        with pytest.raises(c.CholError) as e:
            c.chol_factor(p.h, 0, 96, 0, 96)
        assert e.value.status == -4
        x = torch.zeros((96, 96), dtype=torch.float64, device="cuda")
        with pytest.raises(c.CholError) as e:
            c.chol_factor(p.h, x, 95, x, 96)
        assert e.value.status == -5
