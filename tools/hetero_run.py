"""NEXT-3 measurement: the host CPU cores as a second resource class taking every TRSM at
least d tiles below the diagonal (the paper's static rule, Fig. 11), against
the GPU alone.  Prints one JSON line per (n, d): best of 3 factorization times.
  python tools/hetero_run.py 19200,46080 0,40,30,20"""
import json, os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c

ns = [int(x) for x in sys.argv[1].split(",")] if len(sys.argv) > 1 else [19200]
ds = [int(x) for x in sys.argv[2].split(",")] if len(sys.argv) > 2 else [0, 16, 12, 8]
nb = 960
for n in ns:
    N = n // nb
    for d in ds:
        if d >= N:
            continue
        ntr = sum(1 for k in range(N) for i in range(k + 1, N) if d > 0 and i - k >= d)
        with c.Plan(n, nb, cpu_trsm_distance=d) as p:
            ts = []
            for r in range(4):
                c.chol_generate(p.h, 0, 0)
                t0 = time.perf_counter()
                assert c.chol_factor_inplace(p.h) == 0
                ts.append((c.chol_last_times(p.h)[0], time.perf_counter() - t0))
            best = min(ts[1:])
        print(json.dumps({"n": n, "d": d, "host_trsms": ntr, "ms": round(best[0] * 1e3, 3),
                          "wall_ms": round(best[1] * 1e3, 3), "tflops": round(n ** 3 / 3 / best[0] / 1e12, 3)}),
              flush=True)
