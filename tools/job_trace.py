"""Per-job trace analysis of the persistent scheduler: utilisation over time, per type."""
import sys, os, json
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import paper_conf_ipps_agullobehkmt15_b200 as c

n = int(sys.argv[1]) if len(sys.argv) > 1 else 19200
pol = int(sys.argv[2]) if len(sys.argv) > 2 else 0  # 0 = CP_PRIORITY
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
span = t1.max() - t0.min()
busy = (t1 - t0).sum()
out = {"n": n, "policy": pol, "factor_ms": t_f * 1e3, "span_ms": span / 1e6, "jobs": len(jt), "workers": int(W),
       "utilisation": busy / (W * span)}
for k in range(len(JT)):
    m = typ == k
    if m.any():
        d = (t1[m] - t0[m]) / 1e3
        out[JT[k]] = {"n": int(m.sum()), "mean_us": round(float(d.mean()), 2), "p50_us": round(float(np.median(d)), 2),
                      "max_us": round(float(d.max()), 2), "busy_ms": round(float(d.sum()) / 1e3, 2)}
# gaps between consecutive jobs on the same worker (scheduling overhead)
gaps = []
for w in range(W):
    m = worker == w
    a, b = t0[m], t1[m]
    o = np.argsort(a)
    a, b = a[o], b[o]
    gaps.append(a[1:] - b[:-1])
g = np.concatenate(gaps) / 1e3
out["gap_us"] = {"mean": round(float(g.mean()), 2), "p50": round(float(np.median(g)), 2), "p90": round(float(np.percentile(g, 90)), 2),
                 "total_ms_per_worker": round(float(g.sum()) / W / 1e3, 2)}
# utilisation timeline in 20 bins
edges = np.linspace(t0.min(), t1.max(), 21)
util = []
for i in range(20):
    lo, hi = edges[i], edges[i + 1]
    ov = np.clip(np.minimum(t1, hi) - np.maximum(t0, lo), 0, None).sum()
    util.append(round(float(ov / (W * (hi - lo))), 2))
out["util_timeline"] = util
tq = jt[:, 4].astype(np.int64)
wait = (t0 - tq) / 1e3
for k in range(len(JT)):
    m = typ == k
    if m.any():
        out[JT[k]]["wait_p50_us"] = round(float(np.median(wait[m])), 1)
        out[JT[k]]["wait_p90_us"] = round(float(np.percentile(wait[m], 90)), 1)
# queued (ready, not started) jobs over time, sampled at 20 points
samples = np.linspace(t0.min(), t1.max(), 20)
out["queued_timeline"] = [int(((tq <= s) & (t0 > s)).sum()) for s in samples]
out["running_timeline"] = [int(((t0 <= s) & (t1 > s)).sum()) for s in samples]
print(json.dumps(out))
# long gaps: what job type preceded / followed, and when (fraction of span)
rows = []
for w in range(W):
    m = np.where(worker == w)[0]
    o = m[np.argsort(t0[m])]
    for a, b in zip(o[:-1], o[1:]):
        g = (t0[b] - t1[a]) / 1e3
        if g > 20:
            rows.append((g, JT[typ[a]], JT[typ[b]], round(float((t1[a] - t0.min()) / span), 3), round(float((t0[b] - tq[b]) / 1e3), 1)))
rows.sort(reverse=True)
from collections import Counter
print(json.dumps({"long_gaps": len(rows), "total_long_gap_ms_per_worker": round(sum(r[0] for r in rows) / W / 1e3, 2),
                  "by_prev_next": Counter((r[1], r[2]) for r in rows).most_common(8),
                  "examples(gap_us,prev,next,when,next_wait_us)": rows[:12]}))
