"""Small driver for ncu captures: one factorization (scheduler) and one GEMM batch."""
import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c
n = int(sys.argv[1]) if len(sys.argv) > 1 else 19200
nb = 960
what = sys.argv[2] if len(sys.argv) > 2 else "both"
if what in ("both", "sched"):
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
        c.chol_generate(p.h, 0, 0)
        print("info", c.chol_factor_inplace(p.h), "t", c.chol_last_times(p.h)[0])
if what in ("both", "gemm"):
    with c.Plan(n, nb, executor=c.EXEC_HOST) as p:
        c.chol_generate(p.h, 0, 0)
        N = n // nb
        print("gemm batch ms/task", c.chol_run_batch(p.h, c.GEMM, (N - 1) * (N - 2) // 2, 1))
