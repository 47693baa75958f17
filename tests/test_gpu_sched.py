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


@pytest.mark.parametrize("n,env", [(3840, {}), (7680, {}), (9600, {"CHOL_POTRF_BLOCKDAG": "0"}),
                                   (19200, {}), (5760, {"CHOL_TRSM_TAIL": "0", "CHOL_TRSM_BLOCKS": "1"})])
def test_job_trace_respects_block_level_dag(n, env, monkeypatch):
    """The job trace against the block-level dependencies of Algorithm 1's tile operations
    (chol_job_desc gives each job's blocks): a job starts only after every job that wrote a
    block it reads or overwrites has ended -- in the hybrid block tail, inside the POTRF block
    DAG, across the task-level steps, and for every TRSM decomposition (row slabs, the
    right-looking column steps).  t0 / t1: globaltimer at the compute warps' start / end."""
    c = _lib()
    for k_, v_ in env.items():
        monkeypatch.setenv(k_, v_)
    nb = 960
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, trace=2) as p:
        c.chol_generate(p.h, 1, 0)
        assert c.chol_factor_inplace(p.h) == 0
        jt = c.chol_job_trace(p.h)
        jd = c.chol_job_desc(p.h)
    assert len(jt) == len(jd)
    t0, t1 = jt[:, 0].astype(np.int64), jt[:, 1].astype(np.int64)
    typ = (jt[:, 3] >> np.uint64(32)).astype(np.int64)
    assert np.array_equal(typ, jd[:, 0])
    UPD, TRSM, DIAG, PANEL, PUPD, TS, TU = 0, 1, 2, 3, 4, 5, 6
    from collections import defaultdict
    # last end time of the writers of each block group
    upd = {}                    # (i, j, k, bm, bn) -> t1
    slab_w = defaultdict(int)   # (i, k, slab) -> max t1 of the TRSM jobs writing that row slab
    ts_w = {}                   # (i, k, cb, sl) -> t1
    tu_w = defaultdict(int)     # (i, k, sl, c2) -> max t1 of the TU jobs writing block (sl, c2)
    potrf_end = defaultdict(int)  # k -> max t1 of POTRF_k's jobs
    diag, panel, pupd = {}, {}, {}
    for x in range(len(jd)):
        ty, i, j, k, a, b, cc, _ = (int(v) for v in jd[x])
        if t1[x] == 0:
            continue  # untraced (diagonal-block inverses)
        if ty == UPD:
            upd[(i, j, k, a, b)] = t1[x]
        elif ty == TRSM:
            slab_w[(i, k, a)] = max(slab_w[(i, k, a)], t1[x])
        elif ty == TS:
            ts_w[(i, k, a, b)] = t1[x]
            slab_w[(i, k, b)] = max(slab_w[(i, k, b)], t1[x])
        elif ty == TU:
            tu_w[(i, k, b, cc)] = max(tu_w[(i, k, b, cc)], t1[x])
            slab_w[(i, k, b)] = max(slab_w[(i, k, b)], t1[x])
        elif ty in (DIAG, PANEL, PUPD):
            potrf_end[k] = max(potrf_end[k], t1[x])
            if ty == DIAG:
                diag[(k, a)] = t1[x]
            elif ty == PANEL:
                panel[(k, a, b)] = t1[x]
            else:
                pupd[(k, a, b, cc)] = t1[x]
    nbb = nb // 96
    bad = []
    nchecked = [0]

    def need(x, t_prev, what):
        if t_prev is None:
            return
        nchecked[0] += 1
        if t0[x] < t_prev:
            bad.append((tuple(int(v) for v in jd[x]), what, int(t_prev - t0[x])))

    for x in range(len(jd)):
        ty, i, j, k, a, b, cc, _ = (int(v) for v in jd[x])
        if t1[x] == 0:
            continue
        if ty == UPD:  # C(i, j)[a, b] -= L(i, k)[a, :] L(j, k)[b, :]^T
            need(x, slab_w.get((i, k, a)), "operand slab of L_ik")
            need(x, slab_w.get((j, k, b)), "operand slab of L_jk")
            need(x, upd.get((i, j, k - 1, a, b)), "previous update of the block")
        elif ty == TRSM:  # row slab a of A_ik
            for bn in range(nbb):
                need(x, upd.get((i, k, k - 1, a, bn)), "last update of the slab")
            need(x, potrf_end.get(k), "L_kk")
        elif ty == TS:  # block (b, a) of A_ik, column block a
            need(x, upd.get((i, k, k - 1, b, a)), "last update of the block")
            need(x, tu_w.get((i, k, b, a)), "right-looking updates of the block")
            need(x, diag.get((k, a)), "L_kk diagonal block")
        elif ty == TU:  # block (b, cc) -= X[b, a] L_kk[cc, a]^T
            need(x, ts_w.get((i, k, a, b)), "solved block")
            need(x, upd.get((i, k, k - 1, b, cc)), "last update of the block")
            need(x, panel.get((k, a, cc)), "L_kk off-diagonal block")
        elif ty == DIAG:
            need(x, upd.get((k, k, k - 1, a, a)), "SYRK of the previous step")
            need(x, panel.get((k, a - 1, a)), "panel block feeding the fused update")
            for b2 in range(a):
                need(x, pupd.get((k, b2, a, a)), "inner updates of the block")
        elif ty == PANEL:
            need(x, diag.get((k, a)), "diagonal block")
            need(x, upd.get((k, k, k - 1, b, a)), "SYRK of the previous step")
            for b2 in range(a):
                need(x, pupd.get((k, b2, b, a)), "inner updates of the block")
        elif ty == PUPD:
            need(x, panel.get((k, a, b)), "panel block r")
            need(x, panel.get((k, a, cc)), "panel block q")
            need(x, upd.get((k, k, k - 1, b, cc)), "SYRK of the previous step")
            for b2 in range(a):
                need(x, pupd.get((k, b2, b, cc)), "inner updates of the block")
    assert not bad, bad[:10]
    assert len(upd) > 0 and len(diag) > 0
    # every update job checks its two operand slabs; the inner POTRF and TRSM jobs their blocks
    assert nchecked[0] >= 2 * len(upd) + len(diag), (nchecked[0], len(upd), len(diag))
    # the checks bite: a trace whose start times are all shifted before the end of the
    # first traced job fails them
    t0_saved = t0.copy()
    t0[:] = t1[t1 > 0].min() - 1
    bad.clear()
    for x in range(len(jd)):
        if int(jd[x, 0]) == UPD and t1[x] > 0:
            need(x, slab_w.get((int(jd[x, 1]), int(jd[x, 3]), int(jd[x, 4]))), "operand slab of L_ik")
    t0[:] = t0_saved
    assert bad
