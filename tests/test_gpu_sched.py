"""Device scheduler properties: every task and every CTA job runs
exactly once, the trace respects every edge of the Algorithm 1 DAG, workers never
run two jobs at once, busy time fits in the makespan, and non-SPD inputs terminate
with the right info under every policy."""
import numpy as np
import pytest

import oracle
import spdgen
from oracle import dag as odag

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")


def _lib():
    import paper_conf_ipps_agullobehkmt15_b200 as c
    return c


@pytest.mark.parametrize("policy", [0, 1, 2])
@pytest.mark.parametrize("n,nb", [(1920, 96), (3840, 960), (768, 64)])
@pytest.mark.parametrize("block_tail", [0, 2, 99])
def test_trace_respects_dag(n, nb, policy, block_tail, monkeypatch):
    """block_tail = m: the last m steps use block-level dependencies between tasks (hybrid
    DAG): there a task may start once the producer blocks it reads are
    done, so task-level edges into those steps only guarantee t0(b) >= t0(a) and
    t1(b) >= t1(a); every other edge is strict (t0(b) >= t1(a))."""
    c = _lib()
    N = n // nb
    monkeypatch.setenv("CHOL_BLOCK_TAIL", str(block_tail))
    k0 = N - min(block_tail, N)
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=policy, trace=2) as p:
        c.chol_generate(p.h, 3, 0)
        assert c.chol_factor_inplace(p.h) == 0
        recs, makespan = c.chol_trace(p.h)
        jt = c.chol_job_trace(p.h)
        workers = c.chol_get_info(p.h)["workers"]
    ts, E = odag.edges(N)
    assert len(recs) == len(ts)
    key = {(r["type"], r["i"], r["j"], r["k"]): r for r in recs}
    assert len(key) == len(ts)

    def rec(t):  # chol_trace convention: POTRF (k,k,k), TRSM (i,k,k), SYRK (j,j,k), GEMM (i,j,k)
        if t.type == odag.POTRF:
            return key[(0, t.k, t.k, t.k)]
        if t.type == odag.TRSM:
            return key[(1, t.i, t.k, t.k)]
        if t.type == odag.SYRK:
            return key[(2, t.j, t.j, t.k)]
        return key[(3, t.i, t.j, t.k)]

    trec = [rec(t) for t in ts]
    for r in trec:
        assert r["t1_ns"] >= r["t0_ns"]
    for a, b in E:  # task-level direct dependencies: successor starts after predecessor ends
        if ts[a].k >= k0:  # both in the block-level region
            assert trec[b]["t0_ns"] >= trec[a]["t0_ns"], (ts[a].name, ts[b].name)
            assert trec[b]["t1_ns"] >= trec[a]["t1_ns"], (ts[a].name, ts[b].name)
        else:
            assert trec[b]["t0_ns"] >= trec[a]["t1_ns"], (ts[a].name, ts[b].name)
    # job level: each job once, no overlap on a worker, busy <= workers * span
    t0 = jt[:, 0].astype(np.int64)
    t1 = jt[:, 1].astype(np.int64)
    w = (jt[:, 2] >> np.uint64(32)).astype(np.int64)
    assert np.all(t1 >= t0)
    for worker in np.unique(w):
        m = np.where(w == worker)[0]
        o = m[np.argsort(t0[m])]
        assert np.all(t0[o][1:] >= t1[o][:-1])
    span = t1.max() - t0.min()
    assert (t1 - t0).sum() <= workers * span
    assert makespan > 0


@pytest.mark.parametrize("policy", [0, 1, 2])
def test_non_spd_terminates_with_info(policy):
    c = _lib()
    n, nb = 1920, 96
    L0 = spdgen.integer_L0(n, 5)
    A = spdgen.make_non_spd(spdgen.integer_spd(n, 5), L0, 700, "neg")
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=policy) as p:
        dA = torch.from_numpy(A).cuda()
        assert p.factor(dA) == 701


def test_static_pin_distance_and_workers_options():
    c = _lib()
    n, nb = 3840, 960
    A = spdgen.uniform_spd(n, 2)
    outs = []
    for d, lw in [(1, 4), (2, 16), (0, 8)]:
        with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_STATIC, trsm_pin_distance=d,
                    latency_workers=lw) as p:
            dA = torch.from_numpy(A.copy()).cuda()
            assert p.factor(dA) == 0
            outs.append(dA.cpu().numpy())
    assert all(np.array_equal(outs[0], o) for o in outs[1:])


def test_repeated_factorizations_reuse_plan():
    c = _lib()
    n, nb = 1920, 960
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
        res = []
        for _ in range(3):
            c.chol_generate(p.h, 9, 1)
            assert c.chol_factor_inplace(p.h) == 0
            out = torch.empty((n, n), dtype=torch.float64, device="cuda")
            c.chol_gather(p.h, out, n)
            res.append(out.cpu().numpy())
    assert np.array_equal(res[0], spdgen.integer_L0(n, 9))
    assert all(np.array_equal(res[0], r) for r in res[1:])


@pytest.mark.parametrize("policy", [0, 1, 2])
@pytest.mark.parametrize("n,nb,j0", [(1920, 96, 1000), (7680, 960, 3 * 960 + 37)])
def test_non_spd_leading_columns_are_final(policy, n, nb, j0):
    """chol.h: with info = j, columns < nb*floor((j-1)/nb) of L are valid.  The scheduler
    skips only the jobs of steps >= the failing tile column, so every TRSM_i_k and update
    of an earlier step still runs.  Integer family: those columns are exactly L0's
    (device pointers and the streamed host-pointer path)."""
    c = _lib()
    L0 = spdgen.integer_L0(n, 5)
    A = spdgen.make_non_spd(spdgen.integer_spd(n, 5), L0, j0, "zero")
    cols = (j0 // nb) * nb
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=policy) as p:
        dA = torch.from_numpy(A).cuda()
        assert p.factor(dA) == j0 + 1
        L = dA.cpu().numpy()
        assert np.array_equal(L[:, :cols], L0[:, :cols])
        Lh = np.full_like(A, np.nan)
        assert c.chol_factor(p.h, A, n, Lh, n) == j0 + 1  # host buffers: streamed in / out
        assert np.array_equal(Lh[:, :cols], L0[:, :cols])


def test_non_spd_leading_columns_final_task_level_path():
    """The same contract on the bench's task-level path (N = 17 > 16: per-step POTRF nodes,
    J_TRSM row-slab jobs), failing at a tile boundary deep in the factorization."""
    c = _lib()
    n, nb, j0 = 16320, 960, 12 * 960
    L0 = spdgen.integer_L0(n, 6)
    A = spdgen.make_non_spd(spdgen.integer_spd(n, 6), L0, j0, "neg")
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
        dA = torch.from_numpy(A).cuda()
        assert p.factor(dA) == j0 + 1
        assert torch.equal(dA[:, :j0].cpu(), torch.from_numpy(np.ascontiguousarray(L0[:, :j0])))


def test_injected_priorities_keep_the_factor():
    """NEXT-4: static priorities from an exact task-level schedule (chol_optimal_schedule)
    injected into the device scheduler change only the order in which ready tasks run, never
    the factor (R15); wrong lengths are rejected."""
    c = _lib()
    N, nb = 4, 960
    n = N * nb
    mk, optimal, w, r, _ = c.chol_optimal_schedule(N, [2], [[5e-4, 3.5e-4, 1e-4, 1e-4]])
    assert optimal
    outs = []
    for inject in (False, True):
        with c.Plan(n, nb, executor=c.EXEC_SCHEDULER) as p:
            if inject:
                c.chol_set_task_priorities(p.h, [-x for x in r])
            c.chol_generate(p.h, 3, 0)
            assert c.chol_factor_inplace(p.h) == 0
            L = torch.empty((n, n), dtype=torch.float64, device="cuda")
            c.chol_gather(p.h, L, n)
            outs.append(L.cpu().numpy())
            with pytest.raises(c.CholError) as e:
                c.chol_set_task_priorities(p.h, [0.0] * (len(r) - 1))
            assert e.value.status == -6
    assert np.array_equal(outs[0], outs[1])
    ref, _ = oracle.chol_tiled(spdgen.uniform_spd(n, 3), nb)
    assert oracle.rel_diff(outs[1], ref)["max_rel_floored"] <= 1e-10
