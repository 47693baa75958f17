"""Critical-path breakdown of one POTRF (n = nb, N = 1) from the per-job trace.

For each inner step b of the nested POTRF (DIAG b -> PANEL b -> PUPD b): job durations,
and the hops between them (completion of the last predecessor job -> enqueue of the
successor node -> start of its first job).  Usage: potrf_trace.py [nb] [reps]
"""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import paper_conf_ipps_agullobehkmt15_b200 as c

nb = int(sys.argv[1]) if len(sys.argv) > 1 else 960
reps = int(sys.argv[2]) if len(sys.argv) > 2 else 5
bs = 96 if nb % 96 == 0 else (64 if nb % 64 == 0 else 32)
nbb = nb // bs
with c.Plan(nb, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY, trace=2) as p:
    best = None
    for rep in range(reps):
        c.chol_generate(p.h, 0, 0)
        c.chol_factor_inplace(p.h)
        t = c.chol_last_times(p.h)[0]
        jt = c.chol_job_trace(p.h)
        if best is None or t < best[0]:
            best = (t, jt.copy())
t_f, jt = best
t0, t1, tq = (jt[:, x].astype(np.int64) for x in (0, 1, 4))
base = tq.min()
t0, t1, tq = t0 - base, t1 - base, tq - base
# job order of the builder (sched.cu): DIAG b, PANEL(b, r>b), PUPD(b, r>b, b<q<=r)
idx = 0
steps = []
for b in range(nbb):
    d = idx; idx += 1
    m = nbb - 1 - b
    pan = list(range(idx, idx + m)); idx += m
    nu = m * (m + 1) // 2
    upd = list(range(idx, idx + nu)); idx += nu
    steps.append((d, pan, upd))
assert idx == len(jt), (idx, len(jt))
rows = []
prev_end = 0
for b, (d, pan, upd) in enumerate(steps):
    r = {"b": b, "diag_hop_us": (t0[d] - prev_end) / 1e3, "diag_enq_us": (tq[d] - prev_end) / 1e3,
         "diag_us": (t1[d] - t0[d]) / 1e3}
    if pan:
        r["panel_hop_us"] = (t0[pan].min() - t1[d]) / 1e3
        r["panel_us_max"] = (t1[pan] - t0[pan]).max() / 1e3
        r["panel_span_us"] = (t1[pan].max() - t0[pan].min()) / 1e3
        r["pupd_hop_us"] = (t0[upd].min() - t1[pan].max()) / 1e3
        r["pupd_us_max"] = (t1[upd] - t0[upd]).max() / 1e3
        r["pupd_span_us"] = (t1[upd].max() - t0[upd].min()) / 1e3
        prev_end = t1[upd].max()
    else:
        prev_end = t1[d]
    rows.append({k: round(float(v), 2) if not isinstance(v, int) else v for k, v in r.items()})
tot = {k: round(sum(r.get(k, 0) for r in rows), 1) for k in rows[0] if k != "b"}
print(json.dumps({"nb": nb, "bs": bs, "factor_us": round(t_f * 1e6, 1), "span_us": round((t1.max() - t0.min()) / 1e3, 1),
                  "sum": tot}))
for r in rows:
    print(json.dumps(r))
# critical chain D(b) -> P(b+1,b) -> U(b+1,b+1,b) -> D(b+1): enqueue / start / end (us)
chain = []
for b, (d, pan, upd) in enumerate(steps):
    chain.append(("D%d" % b, d))
    if pan:
        chain.append(("P%d" % b, pan[0]))
        chain.append(("U%d" % b, upd[0]))
prev = None
for name, j in chain:
    w = int(jt[j, 2] >> np.uint64(32))
    print(f"{name:4s} w{w:3d} enq {tq[j]/1e3:8.2f} start {t0[j]/1e3:8.2f} end {t1[j]/1e3:8.2f} dur {(t1[j]-t0[j])/1e3:6.2f}"
          + (f" ready->start {(t0[j]-tq[j])/1e3:5.2f} prev_end->enq {(tq[j]-t1[prev])/1e3:5.2f}" if prev is not None else ""))
    prev = j
# every job of the worker that ran D(1), in start order
names = {}
for b, (d, pan, upd) in enumerate(steps):
    names[d] = "D%d" % b
    for x, j in enumerate(pan):
        names[j] = "P(%d,%d)" % (b + 1 + x, b)
    x = 0
    for r in range(b + 1, nbb):
        for q in range(b + 1, r + 1):
            names[upd[x]] = "U(%d,%d,%d)" % (r, q, b)
            x += 1
w1 = int(jt[steps[1][0], 2] >> np.uint64(32))
mine = [j for j in range(len(jt)) if int(jt[j, 2] >> np.uint64(32)) == w1]
mine.sort(key=lambda j: t0[j])
print("worker", w1)
for j in mine[:40]:
    print(f"  {names[j]:12s} enq {tq[j]/1e3:8.2f} start {t0[j]/1e3:8.2f} end {t1[j]/1e3:8.2f}")
