"""SHA-256 of the n x n factor (nb = 960, CP priority, uniform family seed 0) for the
library CHOL_LIB_OVERRIDE points at: a bitwise A/B of two builds.

  CHOL_LIB_OVERRIDE=variants/x.so python tools/factor_hash.py 3840,19200
"""
import hashlib, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import paper_conf_ipps_agullobehkmt15_b200 as c

for n in [int(x) for x in sys.argv[1].split(",")]:
    with c.Plan(n, 960, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
        c.chol_generate(p.h, 0, 0)
        assert c.chol_factor_inplace(p.h) == 0
        L = torch.empty(n, n, dtype=torch.float64, device="cuda")
        c.chol_gather(p.h, L.data_ptr(), n)
    print(os.environ.get("CHOL_LIB_OVERRIDE", "default"), n,
          hashlib.sha256(L.cpu().numpy().tobytes()).hexdigest()[:16], flush=True)
