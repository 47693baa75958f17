"""Where the persistent scheduler's workers sit idle: idle worker-time per time bin, and
what runs while utilisation is low (head / tail of the factorization)."""
import sys, os, json
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import paper_conf_ipps_agullobehkmt15_b200 as c

n = int(sys.argv[1]) if len(sys.argv) > 1 else 19200
pol = int(sys.argv[2]) if len(sys.argv) > 2 else 0  # 0 = CP_PRIORITY
binus = float(sys.argv[3]) if len(sys.argv) > 3 else 250.0
nb = 960
JT = ["UPD", "TRSM", "DIAG", "PANEL", "PUPD", "TS", "TU", "RECV", "INV", "NOP"]
with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=pol, trace=2) as p:
    for rep in range(2):
        c.chol_generate(p.h, 0, 0)
        c.chol_factor_inplace(p.h)
    t_f = c.chol_last_times(p.h)[0]
    jt = c.chol_job_trace(p.h)
t0, t1 = jt[:, 0].astype(np.int64), jt[:, 1].astype(np.int64)
worker = (jt[:, 2] >> np.uint64(32)).astype(np.int64)
typ = (jt[:, 3] >> np.uint64(32)).astype(np.int64)
W = worker.max() + 1
T0, T1 = t0.min(), t1.max()
edges = np.arange(T0, T1 + binus * 1e3, binus * 1e3)
rows = []
tot_idle = 0.0
for lo, hi in zip(edges[:-1], edges[1:]):
    hi = min(hi, T1)
    ov = np.clip(np.minimum(t1, hi) - np.maximum(t0, lo), 0, None)
    idle = W * (hi - lo) - ov.sum()
    tot_idle += idle
    by = {JT[k]: round(float(ov[typ == k].sum() / (hi - lo)), 1) for k in range(10) if ov[typ == k].sum() > 0}
    rows.append((round(float((lo - T0) / 1e6), 2), round(float(idle / 1e6), 3), by))
print(json.dumps({"n": n, "factor_ms": round(t_f * 1e3, 3), "workers": int(W), "idle_worker_ms": round(tot_idle / 1e6, 1),
                  "idle_frac": round(tot_idle / (W * (T1 - T0)), 4)}))
for r in rows:
    if r[1] > 0.05 * W * binus / 1e3:
        print(json.dumps({"t_ms": r[0], "idle_worker_ms": r[1], "busy_workers_by_type": r[2]}))
