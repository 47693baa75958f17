"""H2D tile-copy rate while the persistent factorization kernel runs (DMA vs compute)."""
import sys, os, time, json
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from cuda.bindings import runtime as rt
import paper_conf_ipps_agullobehkmt15_b200 as c

n, nb = 19200, 960
N = n // nb
nt = N * (N + 1) // 2
A = torch.empty((n, n), dtype=torch.float64, pin_memory=True)
A.fill_(1.0)
d = torch.empty((nt, nb, nb), dtype=torch.float64, device="cuda")
s = rt.cudaStreamCreateWithFlags(rt.cudaStreamNonBlocking)[1]
evs = [rt.cudaEventCreate()[1] for _ in range(nt + 1)]
res = {}
with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
    c.chol_generate(p.h, 0, 0)
    for load in (False, True):
        torch.cuda.synchronize()
        if load:
            c.chol_generate(p.h, 0, 0)
            c.chol_factor_async(p.h)
        rt.cudaEventRecord(evs[0], s)
        t = 0
        for j in range(N):
            for i in range(j, N):
                rt.cudaMemcpy2DAsync(d[t].data_ptr(), nb * 8, A.data_ptr() + (i * nb * n + j * nb) * 8, n * 8,
                                     nb * 8, nb, rt.cudaMemcpyKind.cudaMemcpyHostToDevice, s)
                t += 1
                rt.cudaEventRecord(evs[t], s)
        rt.cudaStreamSynchronize(s)
        if load:
            c.chol_wait(p.h)
        ts = [rt.cudaEventElapsedTime(evs[0], evs[k])[1] for k in (1, 10, 50, 100, 150, nt)]
        res["load" if load else "idle"] = {"ms_at_tiles_1_10_50_100_150_all": [round(x, 2) for x in ts],
                                          "GBps": round(nt * nb * nb * 8 / 1e9 / (ts[-1] / 1e3), 1)}
print(json.dumps(res))
