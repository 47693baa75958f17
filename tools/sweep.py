"""BASELINE configs[2] on 1 GPU: n = 960 N for N in a sweep, CP priority; TF/s, % of FP64
peak, bounds recomputed from this run's calibration (bench.calibrate), makespan/mixed."""
import sys, os, json, types
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c
import bench

Ns = [int(x) for x in sys.argv[1].split(",")] if len(sys.argv) > 1 else [10, 12, 16, 20, 24, 28, 32, 40, 48]
nb = 960
for N in Ns:
    n = N * nb
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
        ts = []
        for r in range(4):
            c.chol_generate(p.h, 0, 0)
            assert c.chol_factor_inplace(p.h) == 0
            if r:
                ts.append(c.chol_last_times(p.h)[0])
        workers = c.chol_get_info(p.h)["workers"]
    t = sum(ts) / len(ts)
    args = types.SimpleNamespace(n=n, nb=nb, policy="cp", seed=0)
    T_lat, T_thr = bench.calibrate(c, args)
    b = c.chol_bounds(n, nb, 1, T_lat, T_thr)
    fl = n ** 3 / 3
    print(json.dumps({"N": N, "n": n, "ms": round(t * 1e3, 3), "tflops": round(fl / t / 1e12, 3),
                      "pct_peak": round(100 * fl / t / 1e12 / bench.FP64_PEAK_TFLOPS, 1),
                      "bounds_ms": {k: round(v * 1e3, 3) for k, v in b.items()},
                      "bound_tflops": {k: round(fl / v / 1e12, 2) for k, v in b.items() if v > 0},
                      "makespan_over_mixed": round(t / b["mixed"], 3)}), flush=True)
