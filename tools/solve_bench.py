"""chol_solve timing at one n: device time of the two sweeps (inverses
cached) and the whole call (host B, copies in and out), per nrhs; achieved HBM rate for
the factor reads (2 sweeps x n^2/2 x 8 bytes) and FP64 rate (2 n^2 nrhs flop)."""
import json, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import paper_conf_ipps_agullobehkmt15_b200 as c
import spdgen

n = int(sys.argv[1]) if len(sys.argv) > 1 else 19200
nrhss = [int(x) for x in sys.argv[2].split(",")] if len(sys.argv) > 2 else [1, 32, 96, 960]
nb = 960
with c.Plan(n, nb) as p:
    c.chol_generate(p.h, 0, 0)
    assert c.chol_factor_inplace(p.h) == 0
    for nrhs in nrhss:
        B0 = spdgen.rhs(n, nrhs, 1)
        ts, tt = [], []
        for r in range(6):
            B = B0.copy()
            c.chol_solve(p.h, B, nrhs, nrhs)
            tot, sw = c.chol_last_solve_times(p.h)
            if r:
                ts.append(sw)
                tt.append(tot)
        sw, tot = min(ts), min(tt)
        lbytes = 2 * (n * n / 2) * 8
        print(json.dumps({"n": n, "nrhs": nrhs, "sweeps_ms": round(sw * 1e3, 4), "total_ms": round(tot * 1e3, 4),
                          "L_read_GBps": round(lbytes / sw / 1e9, 1), "fp64_TFps": round(2.0 * n * n * nrhs / sw / 1e12, 3)}),
              flush=True)
