"""Small factorizations and solves for compute-sanitizer (memcheck / racecheck / synccheck):
  compute-sanitizer --tool memcheck python tools/sanitize_run.py"""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import spdgen
import paper_conf_ipps_agullobehkmt15_b200 as c

CASES = [(1920, 96, dict(policy=c.POLICY_CP_PRIORITY)), (960, 96, dict(policy=c.POLICY_STATIC)),
         (3840, 960, dict(policy=c.POLICY_DYNAMIC)),  # all-TS/TU TRSMs, block DAG
         (7680, 960, dict()),                         # slab TRSMs in inverse form + J_INV
         (5760, 960, dict(cpu_trsm_distance=3))]      # host CPU class (OUT/NOP/IN, host flags)
for n, nb, opts in CASES:
    pol = opts.get("policy", 0)
    A = spdgen.uniform_spd(n, 5)
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, **opts) as p:
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
