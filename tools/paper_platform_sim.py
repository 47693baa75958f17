"""The paper's heterogeneous experiment in simulation (§V-C, Figs. 5-10): a
Mirage-like node -- 9 CPU cores + 3 GPUs (L671-678) -- with the GPU/CPU kernel speedups of
Table I (POTRF 2x, TRSM 11x, SYRK 26x, GEMM 29x, L784-790), nb = 960, N = 4..32.  Per N:
dmda, dmdas, dmdas with GEMM/SYRK forced on GPUs (L1000-1007), dmdas with the best
"TRSMs at least d tiles below the diagonal on CPUs" rule (L1019-1025, best d reported as
in L1079-1081), and the area / mixed LP bounds (L349-404) -- all as GFLOP/s = (n^3/3)/t.

Absolute CPU kernel rates are not in the paper (it prints no timings): a core is taken
at 9.5 GFLOP/s for GEMM/SYRK/TRSM and 4.0 GFLOP/s for POTRF (context: X5650 peak 10.6
GFLOP/s per core).  The curves' shapes, not their absolute values, are the point.
Host-only: runs the library's chol_simulate / chol_lp_bound (no GPU)."""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c

nb = 960
flops = [nb ** 3 / 3 + nb ** 2 / 2 + nb / 6, float(nb) ** 3, nb ** 2 * (nb + 1.0), 2.0 * nb ** 3]
rate = [4.0e9, 9.5e9, 9.5e9, 9.5e9]
speedup = [2.0, 11.0, 26.0, 29.0]
CPU = [f / r for f, r in zip(flops, rate)]
GPU = [t / s for t, s in zip(CPU, speedup)]
workers, times = [9, 3], [CPU, GPU]
Ns = [int(x) for x in sys.argv[1].split(",")] if len(sys.argv) > 1 else [4, 8, 12, 16, 20, 24, 28, 32]
for N in Ns:
    n = N * nb
    gf = lambda t: round((n ** 3 / 3) / t / 1e9, 1)
    row = {"N": N, "n": n}
    row["dmda"] = gf(c.chol_simulate(N, workers, times, policy=c.SIM_DMDA))
    row["dmdas"] = gf(c.chol_simulate(N, workers, times, policy=c.SIM_DMDAS))
    row["dmdas_gemm_syrk_on_gpu"] = gf(c.chol_simulate(N, workers, times, policy=c.SIM_DMDAS, gemm_syrk_class=1))
    best = None
    for d in range(1, N):
        t = c.chol_simulate(N, workers, times, policy=c.SIM_DMDAS, gemm_syrk_class=1, trsm_far_class=0,
                            trsm_far_distance=d)
        if best is None or t < best[0]:
            best = (t, d)
    if best:
        row["dmdas_triangle_trsm_on_cpu"] = gf(best[0])
        row["best_d"] = best[1]
    row["area_bound"] = gf(c.chol_lp_bound(N, workers, times, mixed=False)[0])
    row["mixed_bound"] = gf(c.chol_lp_bound(N, workers, times, mixed=True)[0])
    print(json.dumps(row), flush=True)
