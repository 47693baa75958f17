"""Multi-GPU path on ONE GPU: R logical ranks (one plan each, workers = SMs / R, same
process, plain device pointers instead of IPC) run the distributed persistent schedulers
concurrently; the panel tiles travel between ranks through the RECV jobs exactly as they
would over NVLink.  Checked against the oracle."""
import numpy as np
import pytest

import oracle
import spdgen

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")


def _lib():
    import paper_conf_ipps_agullobehkmt15_b200 as c
    return c


def run_logical(n, nb, p, q, seed=0, family=0, A=None, policy=0):  # 0 = CHOL_POLICY_CP_PRIORITY
    c = _lib()
    R = p * q
    sms = torch.cuda.get_device_properties(0).multi_processor_count
    plans = [c.DistPlan(n, nb, R, r, grid_p=p, grid_q=q, workers=sms // R, policy=policy) for r in range(R)]
    c.DistPlan.connect_local(plans)
    if A is None:
        for pl in plans:
            c.chol_generate(pl.h, seed, family)
    else:
        dA = torch.from_numpy(np.ascontiguousarray(A)).cuda()
        for pl in plans:
            c.chol_scatter(pl.h, dA, n)
    for pl in plans:
        c.chol_factor_async(pl.h)
    infos = [c.chol_wait(pl.h) for pl in plans]
    out = torch.zeros((n, n), dtype=torch.float64, device="cuda")
    for pl in plans:
        c.chol_gather(pl.h, out, n)
    torch.cuda.synchronize()
    for pl in plans:
        pl.close()
    nz = [i for i in infos if i]
    return out.cpu().numpy(), (min(nz) if nz else 0)


@pytest.mark.parametrize("n,nb,p,q", [(1920, 96, 1, 2), (1920, 96, 2, 2), (2880, 96, 1, 3), (3840, 960, 2, 2),
                                      (2304, 96, 2, 4)])
def test_dist_matches_oracle(n, nb, p, q):
    A = spdgen.uniform_spd(n, seed=n + p + q)
    L, info = run_logical(n, nb, p, q, A=A)
    ref, rinfo = oracle.chol_tiled(A, nb)
    assert info == rinfo == 0
    d = oracle.rel_diff(L, ref)
    assert d["max_rel_floored"] <= 1e-10, d
    assert oracle.backward_error(A, L) <= 10.0


@pytest.mark.parametrize("p,q", [(1, 2), (2, 2)])
def test_dist_integer_family_bitwise(p, q):
    n, nb = 1920, 96
    L, info = run_logical(n, nb, p, q, seed=4, family=1)
    assert info == 0
    assert np.array_equal(L, spdgen.integer_L0(n, 4))


def test_dist_bitwise_equals_single_gpu():
    """Reading R15 extended: the distribution does not change any tile's update order."""
    c = _lib()
    n, nb = 1920, 96
    A = spdgen.uniform_spd(n, seed=11)
    L2, _ = run_logical(n, nb, 2, 2, A=A)
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
        dA = torch.from_numpy(A.copy()).cuda()
        assert p.factor(dA) == 0
        L1 = dA.cpu().numpy()
    assert np.array_equal(L1, L2)


def test_dist_non_spd_info():
    n, nb = 1920, 96
    L0 = spdgen.integer_L0(n, 6)
    A = spdgen.make_non_spd(spdgen.integer_spd(n, 6), L0, 1000, "zero")
    _, info = run_logical(n, nb, 2, 2, A=A)
    assert info == 1001


def test_two_processes_share_gpu_through_ipc():
    """The real multi-process path (CUDA IPC export/open of the tile stores and flags,
    peer pulls, publish/watch) with two OS processes on cuda:0."""
    import subprocess
    import sys
    import os
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    r = subprocess.run([sys.executable, os.path.join(root, "tools", "two_proc_one_gpu.py"), "960"],
                       capture_output=True, text=True, timeout=240)
    assert r.returncode == 0, r.stderr[-2000:]
    assert "'infos': [0, 0], 'exact': True" in r.stdout, r.stdout


def _run_logical_device(n, nb, p, q, seed, family, policy=0):  # 0 = CHOL_POLICY_CP_PRIORITY
    """run_logical without the host copy: the gathered factor stays on the device."""
    c = _lib()
    R = p * q
    sms = torch.cuda.get_device_properties(0).multi_processor_count
    plans = [c.DistPlan(n, nb, R, r, grid_p=p, grid_q=q, workers=sms // R, policy=policy) for r in range(R)]
    c.DistPlan.connect_local(plans)
    for pl in plans:
        c.chol_generate(pl.h, seed, family)
    for pl in plans:
        c.chol_factor_async(pl.h)
    infos = [c.chol_wait(pl.h) for pl in plans]
    out = torch.zeros((n, n), dtype=torch.float64, device="cuda")
    for pl in plans:
        c.chol_gather(pl.h, out, n)
    torch.cuda.synchronize()
    for pl in plans:
        pl.close()
    return out, infos


@pytest.mark.parametrize("n,p,q", [(24000, 1, 2), (30720, 2, 2), (38400, 2, 4)])
def test_dist_bench_sizes_bitwise_equal_single_gpu(n, p, q):
    """The bench's multi-GPU workloads (weak scaling: n = 24000 / 30720 / 38400 on 1x2 /
    2x2 / 2x4, nb = 960) as logical ranks: the distributed factor equals the single-plan
    factor bit for bit (R15), and for the integer family it is L0 exactly (band check)."""
    c = _lib()
    nb, seed = 960, 21
    Ld, infos = _run_logical_device(n, nb, p, q, seed, 1)
    assert not any(infos), infos
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as pl:
        c.chol_generate(pl.h, seed, 1)
        assert c.chol_factor_inplace(pl.h) == 0
        Ls = torch.empty((n, n), dtype=torch.float64, device="cuda")
        c.chol_gather(pl.h, Ls, n)
        torch.cuda.synchronize()
    assert torch.equal(Ld, Ls)
    del Ls
    Lb = torch.from_numpy(spdgen.integer_L0_bands(n, seed).astype(np.float64)).cuda()
    idx = torch.arange(n, device="cuda")
    nnz_band = 0
    for o in range(spdgen.BW + 1):
        assert torch.equal(Ld[idx[o:], idx[o:] - o], Lb[o, o:]), o
        nnz_band += int(torch.count_nonzero(Lb[o, o:]))
    assert int(torch.count_nonzero(Ld)) == nnz_band  # nothing outside the band


def _packed_owned(M, nb, owner_ok):
    """Tiles (i, j), i >= j, in Algorithm 1 tile order, kept where owner_ok(i, j), packed."""
    N = M.shape[0] // nb
    return np.concatenate([M[i * nb:(i + 1) * nb, j * nb:(j + 1) * nb].ravel()
                           for i in range(N) for j in range(i + 1) if owner_ok(i, j)])


def test_scatter_gather_tiles_single_and_distributed():
    """chol_scatter_tiles / chol_gather_tiles: the owned tiles, packed in tile order, in and
    out of a single-GPU plan and of each rank of a 2x2 distributed plan; the factor equals
    the oracle's, and a wrong tile count is rejected (-6)."""
    c = _lib()
    n, nb, seed = 1920, 96, 17
    A = spdgen.uniform_spd(n, seed)
    ref, _ = oracle.chol_tiled(A, nb)
    N = n // nb
    # single GPU: every tile is owned
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
        packed = np.ascontiguousarray(_packed_owned(A, nb, lambda i, j: True))
        ntiles = N * (N + 1) // 2
        c.chol_scatter_tiles(p.h, packed, ntiles)
        assert c.chol_factor_inplace(p.h) == 0
        out = np.empty_like(packed)
        c.chol_gather_tiles(p.h, out, ntiles)
        want = _packed_owned(np.tril(ref), nb, lambda i, j: True)
        assert np.max(np.abs(out - want)) <= 1e-10 * np.max(np.abs(want))
        with pytest.raises(c.CholError):
            c.chol_gather_tiles(p.h, out, ntiles - 1)
    # 2 x 2 logical ranks: each rank streams only its own tiles
    R, pg, qg = 4, 2, 2
    sms = torch.cuda.get_device_properties(0).multi_processor_count
    plans = [c.DistPlan(n, nb, R, r, grid_p=pg, grid_q=qg, workers=sms // R, policy=c.POLICY_CP_PRIORITY) for r in range(R)]
    c.DistPlan.connect_local(plans)
    owner = lambda i, j: (i % pg) * qg + (j % qg)  # noqa: E731
    counts = []
    for r, pl in enumerate(plans):
        mine = np.ascontiguousarray(_packed_owned(A, nb, lambda i, j: owner(i, j) == r))
        cnt = mine.size // (nb * nb)
        assert cnt == c.chol_get_dist(pl.h)["nowned"]
        counts.append(cnt)
        c.chol_scatter_tiles(pl.h, mine, cnt)
    for pl in plans:
        c.chol_factor_async(pl.h)
    assert [c.chol_wait(pl.h) for pl in plans] == [0] * R
    for r, pl in enumerate(plans):
        out = np.empty(counts[r] * nb * nb)
        c.chol_gather_tiles(pl.h, out, counts[r])
        want = _packed_owned(np.tril(ref), nb, lambda i, j: owner(i, j) == r)
        assert np.max(np.abs(out - want)) <= 1e-10 * np.max(np.abs(ref))
    for pl in plans:
        pl.close()


@pytest.mark.parametrize("ngpus", [2, 4])
def test_single_process_multi_device_plan(ngpus, monkeypatch):
    """chol_plan(n, nb, ngpus > 1): one process drives ngpus ranks (here all on cuda:0 via
    CHOL_MULTI_ONE_DEVICE=1, SMs / ngpus workers each); device and host pointers; the
    factor equals the single-plan factor bit for bit (R15); the merged trace holds every
    task once, from every rank; solve / per-rank calls are rejected (-8)."""
    monkeypatch.setenv("CHOL_MULTI_ONE_DEVICE", "1")
    c = _lib()
    n, nb = 1920, 96
    N = n // nb
    A = spdgen.uniform_spd(n, 23)
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p1:
        d1 = torch.from_numpy(A.copy()).cuda()
        assert p1.factor(d1) == 0
        ref = d1.cpu().numpy()
    with c.Plan(n, nb, ngpus=ngpus, policy=c.POLICY_CP_PRIORITY, trace=1) as p:
        dA = torch.from_numpy(A.copy()).cuda()
        assert p.factor(dA) == 0
        L = dA.cpu().numpy()
        recs, makespan = c.chol_trace(p.h)
        Lh = np.full_like(A, np.nan)
        assert c.chol_factor(p.h, A.copy(), n, Lh, n) == 0
        with pytest.raises(c.CholError):
            p.solve(np.ones(n))
    assert np.array_equal(L, ref)
    assert np.array_equal(Lh, ref)
    assert len(recs) == N * (N + 1) * (N + 2) // 6
    assert {r["gpu"] for r in recs} == set(range(ngpus))
    assert makespan > 0
    # non-SPD input: LAPACK info from the owning rank
    L0 = spdgen.integer_L0(n, 6)
    B = spdgen.make_non_spd(spdgen.integer_spd(n, 6), L0, 700, "zero")
    with c.Plan(n, nb, ngpus=ngpus) as p:
        assert p.factor(torch.from_numpy(B).cuda()) == 701


def test_watchdog_reports_a_stalled_scheduler():
    """SURVEY §5 failure detection: a distributed rank whose peer never launches would spin
    forever; the host watchdog returns -11 after CHOL_WATCHDOG_S seconds (subprocess: the
    stalled kernel dies with its process)."""
    import os
    import subprocess
    import sys
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    r = subprocess.run([sys.executable, os.path.join(root, "tools", "watchdog_check.py")], capture_output=True,
                       text=True, timeout=240)
    assert "watchdog status -11" in r.stdout, (r.stdout[-1000:], r.stderr[-2000:])
