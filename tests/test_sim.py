"""Platform model (§III-A and §IV-C/§V): the library's LP
bound over resource classes (chol_lp_bound) and its DAG replay under dmda / dmdas and the
static rules (chol_simulate), against the oracle (scipy LP, plain-Python replay) and
against what the mathematics fixes: serial sums, the critical path with unlimited
workers, the related-platform closed form, and "every schedule is at least the bound"."""
import math
import random

import pytest

from oracle import bounds, dag, sim


def _lib():
    import paper_conf_ipps_agullobehkmt15_b200 as c
    return c


TYPES = ("POTRF", "TRSM", "SYRK", "GEMM")
# the paper's platform shape: 9 CPU cores + 3 GPUs (L671-678), Table I speedups (L784-790)
CPU = [1.0, 3.0, 3.0, 6.0]  # nb^3 units: POTRF ~1/3, TRSM 1, SYRK 1, GEMM 2 -- x3 for a core
GPU = [CPU[0] / 2, CPU[1] / 11, CPU[2] / 26, CPU[3] / 29]


def _rand_platform(rng, R):
    workers = [rng.randint(1, 6) for _ in range(R)]
    times = [[rng.uniform(0.1, 5.0) for _ in range(4)] for _ in range(R)]
    return workers, times


@pytest.mark.parametrize("seed", range(12))
@pytest.mark.parametrize("mixed", [False, True])
def test_lp_bound_matches_scipy(seed, mixed):
    c = _lib()
    rng = random.Random(seed)
    R = 1 + seed % 3
    N = rng.choice([1, 2, 4, 7, 12, 30])
    workers, times = _rand_platform(rng, R)
    l, nrt = c.chol_lp_bound(N, workers, times, mixed=mixed)
    ref = bounds.lp_area_mixed(N, {r: dict(zip(TYPES, times[r])) for r in range(R)},
                               {r: workers[r] for r in range(R)}, mixed_chain=mixed)
    assert abs(l - ref) <= 1e-9 * max(1.0, ref)
    # the returned assignment is feasible: every task placed, every class within l
    cnt = bounds.task_counts(N)
    for t, name in enumerate(TYPES):
        assert abs(sum(nrt[r][t] for r in range(R)) - cnt[name]) <= 1e-7 * max(1, cnt[name])
    for r in range(R):
        assert sum(nrt[r][t] * times[r][t] for t in range(4)) <= l * workers[r] * (1 + 1e-9) + 1e-9


def test_lp_closed_forms():
    c = _lib()
    # one class: area = sum N_t T_t / M; mixed = max(area, chain)  (R10, R11)
    T = [3.0, 1.2, 1.1, 2.0]
    for N in (1, 3, 10):
        for M in (1, 4):
            a = c.chol_lp_bound(N, [M], [T], mixed=False)[0]
            assert abs(a - bounds.area(N, dict(zip(TYPES, T)), M)) < 1e-9 * a
            m = c.chol_lp_bound(N, [M], [T], mixed=True)[0]
            assert abs(m - max(a, bounds.chain(N, dict(zip(TYPES, T))))) < 1e-9 * m
    # related platform (L791-797): GPU K times faster on every kernel -> W_cpu / (M_cpu + K M_gpu)
    N, K, Mc, Mg = 8, 7.0, 9, 3
    l = c.chol_lp_bound(N, [Mc, Mg], [CPU, [v / K for v in CPU]], mixed=False)[0]
    W = bounds.area(N, dict(zip(TYPES, CPU)), 1)
    assert abs(l - W / (Mc + K * Mg)) < 1e-9 * l
    # a class that cannot run a type (time < 0) gets none of it
    l, nrt = c.chol_lp_bound(6, [4, 2], [[1, 1, 1, -1], [1, 1, 1, 1]], mixed=False)
    assert nrt[0][3] == 0.0


@pytest.mark.parametrize("policy", [0, 1])
@pytest.mark.parametrize("case", range(10))
def test_simulate_matches_oracle(policy, case):
    c = _lib()
    rng = random.Random(100 + case)
    N = rng.choice([1, 2, 3, 5, 8])
    R = 1 + case % 3
    workers, times = _rand_platform(rng, R)
    # dyadic times: every sum is exact, so both sides see the same ties
    times = [[round(v * 16) / 16 + 0.0625 for v in row] for row in times]
    kw = {}
    if case % 4 == 3 and R >= 2:
        kw = dict(gemm_syrk_class=1, trsm_far_class=0, trsm_far_distance=1 + case % 3)
    mk, recs = c.chol_simulate(N, workers, times, policy=policy, records=True, **kw)
    mk_ref, out = sim.simulate(N, workers, times, policy=policy, **kw)
    assert mk == mk_ref
    ts = dag.tasks(N)
    key = {(t.type, t.i, t.j, t.k): idx for idx, t in enumerate(ts)}
    for r in recs:
        w, cls, t0, t1 = out[key[(r["type"], r["i"], r["j"], r["k"])]]
        assert (r["worker"], r["cls"]) == (w, cls)
        assert r["t0_ns"] == round(t0 * 1e9) and r["t1_ns"] == round(t1 * 1e9)


def test_simulate_serial_and_unlimited():
    c = _lib()
    T = [3.0, 1.25, 1.5, 2.0]
    for N in (1, 4, 9):
        cnt = bounds.task_counts(N)
        serial = sum(cnt[n] * T[t] for t, n in enumerate(TYPES))
        for pol in (0, 1):
            assert c.chol_simulate(N, [1], [T], policy=pol) == serial
            # more workers than tasks: every task starts when ready -> the critical path
            big = c.chol_simulate(N, [len(dag.tasks(N))], [T], policy=pol)
            assert abs(big - bounds.critical_path(N, dict(zip(TYPES, T)))) < 1e-9
    # unit weights: the 3N-2 chain of P:L383-386
    assert c.chol_simulate(7, [1000], [[1, 1, 1, 1]], policy=1) == 3 * 7 - 2


@pytest.mark.parametrize("N", [2, 6, 12])
def test_simulated_schedules_respect_dag_and_bounds(N):
    c = _lib()
    workers, times = [9, 3], [CPU, GPU]
    l_mixed = c.chol_lp_bound(N, workers, times, mixed=True)[0]
    ts, E = dag.edges(N)
    key = {(t.type, t.i, t.j, t.k): idx for idx, t in enumerate(ts)}
    for pol in (0, 1):
        for rule in ({}, dict(gemm_syrk_class=1), dict(gemm_syrk_class=1, trsm_far_class=0, trsm_far_distance=2)):
            mk, recs = c.chol_simulate(N, workers, times, policy=pol, records=True, **rule)
            assert mk >= l_mixed * (1 - 1e-12)  # the LP is a lower bound of any schedule
            by = {key[(r["type"], r["i"], r["j"], r["k"])]: r for r in recs}
            for a, b in E:
                assert by[b]["t0_ns"] >= by[a]["t1_ns"]
            per_w = {}
            for r in recs:
                per_w.setdefault(r["worker"], []).append((r["t0_ns"], r["t1_ns"]))
                assert abs((r["t1_ns"] - r["t0_ns"]) - times[r["cls"]][r["type"]] * 1e9) <= 2
                if rule.get("gemm_syrk_class") is not None and r["type"] in (dag.SYRK, dag.GEMM):
                    assert r["cls"] == 1
                if rule.get("trsm_far_class") is not None and r["type"] == dag.TRSM and \
                        r["i"] - r["k"] >= rule["trsm_far_distance"]:
                    assert r["cls"] == 0
            for iv in per_w.values():
                iv.sort()
                assert all(iv[q][0] >= iv[q - 1][1] for q in range(1, len(iv)))


def test_simulate_errors():
    c = _lib()
    with pytest.raises(c.CholError):
        c.chol_simulate(0, [1], [[1, 1, 1, 1]])
    with pytest.raises(c.CholError):  # no class may run GEMM
        c.chol_simulate(4, [1], [[1, 1, 1, -1]])
    with pytest.raises(c.CholError):
        c.chol_lp_bound(4, [1], [[1, 1, 1, math.inf]])
