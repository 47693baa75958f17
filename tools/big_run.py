"""BASELINE configs[3]'s matrix (n = 92160, 96 x 96 tiles of nb = 960) on ONE GPU: timing
(persistent scheduler, CP priority) and an exactness check with the integer family
(L must be L0 bit for bit: band compared, everything else exactly 0)."""
import json, os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import paper_conf_ipps_agullobehkmt15_b200 as c
import spdgen

n = int(sys.argv[1]) if len(sys.argv) > 1 else 92160
nb = 960
out = {"n": n, "nb": nb, "tasks": None}
with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
    ts = []
    for r in range(3):
        c.chol_generate(p.h, 0, 0)
        assert c.chol_factor_inplace(p.h) == 0
        if r:
            ts.append(c.chol_last_times(p.h)[0])
    out["ms"] = [round(t * 1e3, 2) for t in ts]
    out["tflops"] = round(n ** 3 / 3 / min(ts) / 1e12, 3)
    out["pct_peak"] = round(100 * n ** 3 / 3 / min(ts) / 1e12 / 37.1, 1)
    seed = 5
    c.chol_generate(p.h, seed, 1)
    assert c.chol_factor_inplace(p.h) == 0
    L = torch.empty((n, n), dtype=torch.float64, device="cuda")
    c.chol_gather(p.h, L, n)
    torch.cuda.synchronize()
Lb = torch.from_numpy(spdgen.integer_L0_bands(n, seed).astype(np.float64)).cuda()
idx = torch.arange(n, device="cuda")
ok, nnz = True, 0
for o in range(spdgen.BW + 1):
    ok &= bool(torch.equal(L[idx[o:], idx[o:] - o], Lb[o, o:]))
    nnz += int(torch.count_nonzero(Lb[o, o:]))
out["integer_family_exact"] = ok and int(torch.count_nonzero(L)) == nnz
print(json.dumps(out), flush=True)
