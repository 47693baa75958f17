"""Scheduler policies timing + trace summary (development tool)."""
import sys, json, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import paper_conf_ipps_agullobehkmt15_b200 as c

def summarize(recs, ms):
    busy = {}
    for r in recs:
        busy.setdefault(c.TYPE_NAMES[r["type"]], []).append((r["t1_ns"] - r["t0_ns"]) / 1e3)
    return {k: {"n": len(v), "mean_us": round(float(np.mean(v)), 1), "max_us": round(float(np.max(v)), 1)} for k, v in busy.items()}

n = int(sys.argv[1]) if len(sys.argv) > 1 else 19200
nb = 960
for pol in (0, 1, 2):
    for ex in (c.EXEC_SCHEDULER,):
        with c.Plan(n, nb, executor=ex, policy=pol, trace=1) as p:
            ts = []
            for rep in range(3):
                c.chol_generate(p.h, 0, 0)
                info = c.chol_factor_inplace(p.h)
                ts.append(c.chol_last_times(p.h)[0])
            recs, mk = c.chol_trace(p.h)
            # critical chain: POTRF_k start/end
            pot = [(r["k"], r["t0_ns"] / 1e6, r["t1_ns"] / 1e6) for r in recs if r["type"] == 0]
            print(json.dumps({"n": n, "policy": pol, "info": info, "s": min(ts), "tflops": n**3/3/min(ts)/1e12,
                              "makespan_ms": mk * 1e3, "types": summarize(recs, mk),
                              "potrf_ms": [(k, round(a, 2), round(b, 2)) for k, a, b in pot][:6]}))
