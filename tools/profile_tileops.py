"""One launch of each host-executor tile-op kernel for ncu (GEMM batch, SYRK batch, TRSM
batch, POTRF inner kernels) at nb = 960."""
import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c
n, nb = 9600, 960
N = n // nb
with c.Plan(n, nb, executor=c.EXEC_HOST) as p:
    c.chol_generate(p.h, 0, 0)
    c.chol_run_batch(p.h, c.GEMM, (N - 1) * (N - 2) // 2, 1)
    c.chol_run_batch(p.h, c.SYRK, N - 1, 1)
    c.chol_generate(p.h, 0, 0)
    c.chol_run_batch(p.h, c.POTRF, N, 1)
    c.chol_run_batch(p.h, c.TRSM, N - 1, 1)
