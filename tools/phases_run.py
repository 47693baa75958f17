"""Driver for the CHOL_PHASES instrumented library (tools/build_variant.sh phases -DCHOL_PHASES):
one factorization, or one GEMM batch through the persistent scheduler, at n; the library
prints the per-job phase cycles of the K = nb GEMM/SYRK jobs on chol_destroy (stderr).
  CHOL_LIB_OVERRIDE=variants/phases.so python tools/phases_run.py factor 46080
  CHOL_LIB_OVERRIDE=variants/phases.so python tools/phases_run.py batch 46080 [count]"""
import os
import sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c

mode, n = sys.argv[1], int(sys.argv[2])
nb = 960
N = n // nb
with c.Plan(n, nb, executor=c.EXEC_SCHEDULER) as p:
    c.chol_generate(p.h, 0, 0)
    if mode == "factor":
        assert c.chol_factor_inplace(p.h) == 0
        print(mode, n, "ms", c.chol_last_times(p.h)[0] * 1e3, flush=True)
    else:
        cnt = int(sys.argv[3]) if len(sys.argv) > 3 else (N - 1) * (N - 2) // 2
        print(mode, n, cnt, "us/task", c.chol_run_batch(p.h, c.GEMM, cnt, 1) * 1e3, flush=True)
