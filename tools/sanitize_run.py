"""Small factorizations and solves for compute-sanitizer (memcheck / racecheck / synccheck):
  compute-sanitizer --tool memcheck python tools/sanitize_run.py"""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import spdgen
import paper_conf_ipps_agullobehkmt15_b200 as c

for n, nb, pol in [(1920, 96, 1), (960, 96, 2), (3840, 960, 0)]:
    A = spdgen.uniform_spd(n, 5)
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=pol) as p:
        dA = torch.from_numpy(A.copy()).cuda()
        assert p.factor(dA) == 0
        torch.cuda.synchronize()
        L = dA.cpu().numpy()
        B = spdgen.rhs(n, 3, 1)
        X = B.copy()
        p.solve(X)
        X1 = B[:, :1].copy()
        p.solve(X1)
    ref = np.linalg.cholesky(A)  # LAPACK; the oracle is test infrastructure only
    rel = float(np.max(np.abs(L - ref)) / np.max(np.abs(ref)))
    print(n, nb, pol, "max_rel", rel, flush=True)
    assert rel <= 1e-10
print("sanitize run ok")
