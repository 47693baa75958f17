"""Two PROCESSES sharing cuda:0 run one distributed factorization through CUDA IPC (the
exact multi-GPU code path: IPC handle export/open, peer pulls, publish flags).  Without
MPS the two persistent kernels time-slice, so this is a correctness check, not a timing."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np


def worker(rank, world, port, n, nb, q):
    import torch
    import torch.distributed as dist
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    torch.cuda.set_device(0)
    import paper_conf_ipps_agullobehkmt15_b200 as c

    def allgather(b):
        out = [None] * world
        dist.all_gather_object(out, b)
        return out

    plan = c.DistPlan(n, nb, world, rank, allgather=allgather, grid_p=1, grid_q=world, workers=74, policy=c.POLICY_CP_PRIORITY)
    c.chol_generate(plan.h, 2, 1)
    dist.barrier()
    t0 = time.time()
    info = c.chol_factor_inplace(plan.h)
    out = torch.zeros((n, n), dtype=torch.float64, device="cuda")
    c.chol_gather(plan.h, out, n)
    torch.cuda.synchronize()
    q.put((rank, info, out.cpu().numpy(), time.time() - t0))
    dist.barrier()
    plan.close()
    dist.destroy_process_group()


if __name__ == "__main__":
    import torch.multiprocessing as mp
    import spdgen
    n, nb = int(sys.argv[1]) if len(sys.argv) > 1 else 960, 96
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = 29600 + os.getpid() % 1000
    ps = [ctx.Process(target=worker, args=(r, 2, port, n, nb, q)) for r in range(2)]
    for p in ps:
        p.start()
    res = sorted([q.get(timeout=300) for _ in ps], key=lambda x: x[0])
    for p in ps:
        p.join(timeout=60)
    L = res[0][2] + res[1][2]  # disjoint owned tiles (rank 0 also zeroed the upper part)
    print({"infos": [r[1] for r in res], "exact": bool(np.array_equal(L, spdgen.integer_L0(n, 2))),
           "secs": [round(r[3], 3) for r in res]})
