"""Quick GPU smoke/timing used during development."""
import sys, time, json, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import paper_conf_ipps_agullobehkmt15_b200 as c

ex = int(sys.argv[1]) if len(sys.argv) > 1 else c.EXEC_HOST
for n, nb in [(9600, 960), (19200, 960)]:
    with c.Plan(n, nb, executor=ex) as p:
        for rep in range(3):
            c.chol_generate(p.h, 0, 0)
            info = c.chol_factor_inplace(p.h)
            f, _ = c.chol_last_times(p.h)
            print(json.dumps({"n": n, "nb": nb, "exec": ex, "info": info, "s": f, "tflops": n**3/3/f/1e12}))
    with c.Plan(3*nb, nb, executor=c.EXEC_HOST) as p:
        c.chol_generate(p.h, 0, 0)
        for t, name in enumerate(c.TYPE_NAMES):
            ms = c.chol_run_task(p.h, t, 2, 1, 0, 5)
            print(json.dumps({"task": name, "lat_ms": ms}))
    with c.Plan(n, nb, executor=c.EXEC_HOST) as p:
        c.chol_generate(p.h, 0, 0)
        N = n // nb
        for t, cnt in [(0, N), (1, N - 1), (2, N - 1), (3, (N - 1) * (N - 2) // 2)]:
            ms = c.chol_run_batch(p.h, t, cnt, 2)
            fl = [nb**3/3, nb**3, nb**3, 2*nb**3][t]
            print(json.dumps({"batch": c.TYPE_NAMES[t], "count": cnt, "thr_ms": ms, "tflops": fl/ms/1e9}))
