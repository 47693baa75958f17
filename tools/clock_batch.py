"""SM clocks / power under a saturating GEMM batch through the persistent scheduler vs under
the factorization itself (nvidia-smi sampled every 200 ms, bench.ClockSampler): does the
calibration batch run at the factorization's clock?  usage: python tools/clock_batch.py [n]"""
import json, os, sys
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import bench
import paper_conf_ipps_agullobehkmt15_b200 as c

n = int(sys.argv[1]) if len(sys.argv) > 1 else 46080
nb = 960
N = n // nb
with c.Plan(n, nb) as p:
    c.chol_generate(p.h, 0, 0)
    with bench.ClockSampler(0) as clk:
        us = c.chol_run_batch(p.h, c.GEMM, (N - 1) * (N - 2) // 2, 30) * 1e3
    print(json.dumps({"what": "GEMM batch", "n": n, "us_per_task": us, "clocks": clk.summary()}), flush=True)
    ts = []
    with bench.ClockSampler(0) as clk:
        for _ in range(4):
            c.chol_generate(p.h, 0, 0)
            c.chol_factor_inplace(p.h)
            ts.append(c.chol_last_times(p.h)[0])
    print(json.dumps({"what": "factorization", "n": n, "ms": [t * 1e3 for t in ts], "clocks": clk.summary()}),
          flush=True)
