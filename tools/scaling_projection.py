"""Multi-GPU projection from one-GPU measurements (host only, no GPU): for a p x q 2D
block-cyclic grid, the owner-area bound (the busiest rank's summed per-task throughput times,
`chol_owner_area`), the chain bound (`chol_bounds`), the remote panel tiles each rank pulls
(`chol_dist_layout`) and their transfer time at a given per-GPU NVLink rate.  The per-task
times come from a bench line's R9 calibration (profiles/r02/bench_r02.json).  A projection,
not a measurement: the pool offers one GPU.
  python tools/scaling_projection.py [bench.json] [GB/s per GPU]"""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
bench = json.load(open(sys.argv[1] if len(sys.argv) > 1 else os.path.join(ROOT, "profiles", "r02", "bench_r02.json")))
link = float(sys.argv[2]) if len(sys.argv) > 2 else 900.0  # GB/s into one GPU (NVLink 5, one direction)
T_lat = [bench["bounds"]["T_lat_s"][k] for k in ("POTRF", "TRSM", "SYRK", "GEMM")]
T_thr = [bench["bounds"]["T_thr_s"][k] for k in ("POTRF", "TRSM", "SYRK", "GEMM")]
t1_meas = bench["ms_per_step"] / 1e3
nb = 960
for n in (46080, 92160):
    N = n // nb
    b1 = c.chol_bounds(n, nb, 1, T_lat, T_thr)
    eff = b1["area"] / t1_meas if n == bench["config"]["n"] else None  # area bound / measured (1 GPU)
    for (p, q) in ((1, 1), (1, 2), (2, 2), (2, 4)):
        M = p * q
        area, per = c.chol_owner_area(N, p, q, T_thr)
        pulled = max(c.chol_dist_layout(n, nb, p, q, r)[1] for r in range(M)) if M > 1 else 0
        comm_s = pulled * nb * nb * 8 / (link * 1e9)
        bound = max(area, b1["chain"])
        row = {"n": n, "gpus": M, "grid": f"{p}x{q}", "owner_area_ms": round(area * 1e3, 2),
               "chain_ms": round(b1["chain"] * 1e3, 2), "imbalance": round(area * M / sum(per), 4),
               "tiles_pulled_busiest_rank": pulled, "pull_ms_at_link": round(comm_s * 1e3, 2),
               "speedup_bound_vs_1gpu_bound": round(max(b1["area"], b1["chain"]) / bound, 2)}
        if eff:
            # the one-GPU makespan / area ratio carried over to every rank
            row["projected_ms"] = round(max(area / eff, b1["chain"]) * 1e3, 1)
            row["projected_speedup"] = round(t1_meas / max(area / eff, b1["chain"]), 2)
        print(json.dumps(row), flush=True)
