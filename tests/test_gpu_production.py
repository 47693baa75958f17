"""Element-wise oracle parity on the code paths the bench actually runs.

The whole-factorization cases of test_gpu_parity.py have N <= 4 (all of the DAG is the
block-level tail) or nb = 96 (one block per tile).  Here every case is nb = 960 on the
uniform family, compared with oracle.chol_tiled element by element (floored relative
difference <= 1e-10, reading R8) plus the backward error (<= 10):

* the bench configuration itself, n = 19200 (N = 20: per-step POTRF nodes, J_TRSM row-slab
  jobs with producer-streamed K chunks, the block tail), device pointers AND the streamed
  host-pointer chol_factor, every policy (bitwise equal to each other, reading R15), the
  host-sequenced executor, and 2x2 / 1x2 logical ranks of the distributed path;
* N = 5 / 7 / 9 with the scheduler's development switches forcing each decomposition
  (task-level POTRF, slab TRSMs everywhere, right-looking TRSM blocks, per-slab chains, the
  blocked tail with slab TRSMs, unfused POTRF chain updates).

The oracle factors n = 19200 in ~100 s on the GPU box's 16 host cores (once per module)."""
import numpy as np
import pytest

import oracle
import spdgen

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")

NB = 960


def _lib():
    import paper_conf_ipps_agullobehkmt15_b200 as c
    return c


_ORACLE = {}


def _oracle(n, seed):
    if (n, seed) not in _ORACLE:
        A = spdgen.uniform_spd(n, seed)
        ref, info = oracle.chol_tiled(A, NB)
        assert info == 0
        _ORACLE[(n, seed)] = (A, ref)
    return _ORACLE[(n, seed)]


def _check(A, L, ref):
    d = oracle.rel_diff(L, ref)
    assert d["max_rel_floored"] <= 1e-10, d
    assert np.all(np.triu(L, 1) == 0.0)
    assert oracle.backward_error(A, L) <= 10.0


def _factor_device(c, A, **opts):
    n = A.shape[0]
    with c.Plan(n, NB, **opts) as p:
        dA = torch.from_numpy(A).cuda()
        info = p.factor(dA)
        torch.cuda.synchronize()
        assert info == 0
        return dA.cpu().numpy()


# ----------------------------------------------------------------------------- the bench config
@pytest.fixture(scope="module")
def bench19200():
    return _oracle(19200, 0)


def test_bench_config_device_pointers_all_policies(bench19200):
    c = _lib()
    A, ref = bench19200
    Ls = [_factor_device(c, A, policy=pol) for pol in (c.POLICY_CP_PRIORITY, c.POLICY_DYNAMIC, c.POLICY_STATIC)]
    _check(A, Ls[0], ref)
    for L in Ls[1:]:  # reading R15: the schedule does not change any tile's update order
        assert np.array_equal(L, Ls[0])


def test_bench_config_streamed_host_pointers(bench19200):
    """chol_factor with HOST buffers: tiles streamed in during the factorization (arrival
    flags), every final tile streamed out as it is published -- the bench's e2e path."""
    c = _lib()
    A, ref = bench19200
    n = A.shape[0]
    with c.Plan(n, NB) as p:
        L = np.full_like(A, np.nan)
        assert c.chol_factor(p.h, A, n, L, n) == 0
        _check(A, L, ref)
        # in place on the host (A == L), the bench's single-buffer e2e form
        B = A.copy()
        assert c.chol_factor(p.h, B, n, B, n) == 0
        assert np.array_equal(B, L)


def test_bench_config_host_executor(bench19200):
    c = _lib()
    A, ref = bench19200
    _check(A, _factor_device(c, A, executor=c.EXEC_HOST), ref)


@pytest.mark.parametrize("p,q", [(2, 2), (1, 2)])
def test_bench_config_distributed_logical_ranks(bench19200, p, q):
    """The multi-GPU path (RECV jobs over peer memory, publish / watch flags) at the bench
    size, uniform family, against the oracle -- and bitwise equal to the single plan."""
    c = _lib()
    A, ref = bench19200
    n = A.shape[0]
    R = p * q
    sms = torch.cuda.get_device_properties(0).multi_processor_count
    plans = [c.DistPlan(n, NB, R, r, grid_p=p, grid_q=q, workers=sms // R) for r in range(R)]
    c.DistPlan.connect_local(plans)
    dA = torch.from_numpy(A).cuda()
    for pl in plans:
        c.chol_scatter(pl.h, dA, n)
    for pl in plans:
        c.chol_factor_async(pl.h)
    assert [c.chol_wait(pl.h) for pl in plans] == [0] * R
    out = torch.zeros((n, n), dtype=torch.float64, device="cuda")
    for pl in plans:
        c.chol_gather(pl.h, out, n)
    torch.cuda.synchronize()
    for pl in plans:
        pl.close()
    L = out.cpu().numpy()
    _check(A, L, ref)
    assert np.array_equal(L, _factor_device(c, A))


# ----------------------------------------------------------------------------- forced decompositions
SWITCHES = {
    "task_level_potrf": {"CHOL_BLOCK_TAIL": "0", "CHOL_POTRF_BLOCKDAG": "0", "CHOL_POTRF0_BLOCKDAG": "0"},
    "slab_trsm_everywhere": {"CHOL_TRSM_TAIL": "0", "CHOL_BLOCK_TAIL": "0"},
    "right_looking_trsm": {"CHOL_TRSM_BLOCKS": "1", "CHOL_BLOCK_TAIL": "0"},
    "slab_chain_trsm": {"CHOL_TRSM_SLABCHAIN": "1", "CHOL_TRSM_TAIL": "3", "CHOL_BLOCK_TAIL": "0"},
    "tail_slab_trsm_unfused": {"CHOL_TAIL_TRSM": "1", "CHOL_POTRF_FUSE": "0", "CHOL_BLOCK_TAIL": "3"},
    "defaults": {},
}


@pytest.mark.parametrize("N", [5, 7, 9])
@pytest.mark.parametrize("switch", list(SWITCHES))
def test_forced_decompositions_match_oracle(N, switch, monkeypatch):
    for k, v in SWITCHES[switch].items():
        monkeypatch.setenv(k, v)
    c = _lib()
    A, ref = _oracle(N * NB, N)
    _check(A, _factor_device(c, A), ref)


@pytest.mark.parametrize("N,d", [(8, 3), (12, 6)])
def test_host_cpu_class_trsms_match_oracle(N, d, monkeypatch):
    """NEXT-3: the TRSMs at least d tiles below the diagonal run on the host CPU cores (the
    paper's static rule); the factor still matches the oracle, device and streamed host
    pointers, and the integer family stays exact."""
    c = _lib()
    A, ref = _oracle(N * NB, N + 100)
    n = A.shape[0]
    with c.Plan(n, NB, cpu_trsm_distance=d) as p:
        dA = torch.from_numpy(A).cuda()
        assert p.factor(dA) == 0
        _check(A, dA.cpu().numpy(), ref)
        L = np.full_like(A, np.nan)
        assert c.chol_factor(p.h, A, n, L, n) == 0
        _check(A, L, ref)
        c.chol_generate(p.h, 4, 1)
        assert c.chol_factor_inplace(p.h) == 0
        out = torch.empty((n, n), dtype=torch.float64, device="cuda")
        c.chol_gather(p.h, out, n)
        assert np.array_equal(out.cpu().numpy(), spdgen.integer_L0(n, 4))
