"""Multi-GPU host logic (CPU only): the 2D block-cyclic owner map and
the set of remote panel tiles each rank must receive, checked against the oracle's task
graph; plus a world_size-2 gloo run that exchanges the layouts between processes."""
import os

import pytest
import torch.multiprocessing as mp

from oracle import dag as odag


def _chol():
    from paper_conf_ipps_agullobehkmt15_b200 import build
    build.build()
    import paper_conf_ipps_agullobehkmt15_b200 as c
    return c


def owner(i, j, p, q):
    return (i % p) * q + (j % q)


def expected_needs(N, p, q, rank):
    """Remote tiles read by the tasks this rank owns (owner-computes), from the oracle DAG."""
    need = set()
    for t in odag.tasks(N):
        wi, wj = t.writes
        if owner(wi, wj, p, q) != rank:
            continue
        for (ri, rj) in t.reads:
            if owner(ri, rj, p, q) != rank:
                need.add((ri, rj))
    return need


@pytest.mark.parametrize("N,p,q", [(5, 1, 2), (8, 2, 2), (10, 2, 4), (7, 1, 3), (12, 4, 2)])
def test_layout_matches_oracle_dag(N, p, q):
    c = _chol()
    nb = 32
    owned_all = set()
    for rank in range(p * q):
        nowned, ncached, sm = c.chol_dist_layout(N * nb, nb, p, q, rank)
        tiles = [(i, j) for i in range(N) for j in range(i + 1)]
        owned = {tj for t, tj in enumerate(tiles) if 0 <= sm[t] < nowned}
        cached = {tj for t, tj in enumerate(tiles) if sm[t] >= nowned}
        assert owned == {(i, j) for (i, j) in tiles if owner(i, j, p, q) == rank}
        assert not owned & owned_all
        owned_all |= owned
        need = expected_needs(N, p, q, rank)
        assert cached == need
        # remote reads are only final panel tiles L_kk, L_ik (never a tile still being updated)
        slots = sorted(sm[t] for t in range(len(tiles)) if sm[t] >= 0)
        assert slots == list(range(nowned + ncached))
    assert len(owned_all) == N * (N + 1) // 2


def _worker(rank, world, N, p, q, port, out):
    import torch.distributed as dist
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    c = _chol()
    nb = 32
    nowned, ncached, sm = c.chol_dist_layout(N * nb, nb, p, q, rank)
    layouts = [None] * world
    dist.all_gather_object(layouts, (rank, nowned, ncached, sm))
    ok = True
    tiles = [(i, j) for i in range(N) for j in range(i + 1)]
    for (r, no, nc, m) in layouts:
        for t, (i, j) in enumerate(tiles):
            if no <= m[t]:  # r receives tile t: its owner must hold it in an owned slot
                o = owner(i, j, p, q)
                ok &= o != r and 0 <= layouts[o][3][t] < layouts[o][1]
    dist.barrier()
    dist.destroy_process_group()
    out.put((rank, ok))


def test_gloo_two_ranks_exchange_layouts():
    ctx = mp.get_context("spawn")
    q_ = ctx.Queue()
    port = 29500 + os.getpid() % 1000
    procs = [ctx.Process(target=_worker, args=(r, 2, 9, 1, 2, port, q_)) for r in range(2)]
    for pr in procs:
        pr.start()
    res = [q_.get(timeout=120) for _ in procs]
    for pr in procs:
        pr.join(timeout=60)
    assert sorted(res) == [(0, True), (1, True)]
