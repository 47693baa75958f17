"""Tile size sweep at fixed n (CP priority): how the tile size trades the chain (latency)
against per-task efficiency.  Usage: nb_sweep.py n nb1,nb2,..."""
import json, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c
n = int(sys.argv[1])
for nb in [int(x) for x in sys.argv[2].split(",")]:
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
        ts = []
        for r in range(4):
            c.chol_generate(p.h, 0, 0)
            assert c.chol_factor_inplace(p.h) == 0
            if r:
                ts.append(c.chol_last_times(p.h)[0])
    t = min(ts)
    print(json.dumps({"n": n, "nb": nb, "ms": round(t * 1e3, 3), "tflops": round(n ** 3 / 3 / t / 1e12, 3)}), flush=True)
