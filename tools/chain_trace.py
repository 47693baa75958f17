"""Critical chain of one factorization from the per-job trace (development tool).

Walks back from the last job to end: a node is enqueued when its last predecessor
completes, so the job that ended last before a job's enqueue time is taken as the
predecessor that released it.  Prints the chain's time split by job type (work) and
by gaps (enqueue -> start, end -> enqueue of the successor).
Usage: chain_trace.py N [reps] [--list]"""
import json
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import faulthandler
faulthandler.dump_traceback_later(int(os.environ.get('CHAIN_TB', '0')) or 10**6, exit=True)
import paper_conf_ipps_agullobehkmt15_b200 as c

JT = {0: "UPD", 1: "TRSM", 2: "DIAG", 3: "PANEL", 4: "PUPD", 5: "TS", 6: "TU", 7: "RECV", 8: "INV", 9: "NOP"}
N = int(sys.argv[1]) if len(sys.argv) > 1 else 10
reps = int(sys.argv[2]) if len(sys.argv) > 2 and sys.argv[2].isdigit() else 5
nb = 960
n = N * nb
with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY, trace=2) as p:
    best = None
    for rep in range(reps):
        c.chol_generate(p.h, 0, 0)
        assert c.chol_factor_inplace(p.h) == 0
        print('rep', rep, flush=True, file=sys.stderr)
        t = c.chol_last_times(p.h)[0]
        jt = c.chol_job_trace(p.h)
        if rep and (best is None or t < best[0]):
            best = (t, jt.copy())
t_f, jt = best
jt = jt[jt[:, 1] > 0]  # untraced jobs (INV: no paper task) carry no times
t0, t1, tq = (jt[:, x].astype(np.int64) for x in (0, 1, 4))
typ = (jt[:, 3] >> np.uint64(32)).astype(np.int64)
base = min(tq.min(), t0.min())
t0, t1, tq = t0 - base, t1 - base, tq - base
order = np.argsort(t1)
t1s = t1[order]
j = int(np.argmax(t1))
chain = []
while True:
    chain.append(j)
    lim = min(tq[j], t0[j])  # enqueue of the job's node (a job is never started before it)
    k = np.searchsorted(t1s, lim, side="right") - 1
    if k < 0 or len(chain) > len(jt):
        break
    pj = int(order[k])
    if t1[pj] >= t1[j] or pj == j:
        break
    j = pj
chain.reverse()
work, wait, hop = {}, 0, 0
for a, b in zip(chain, chain[1:] + [None]):
    nm = JT.get(int(typ[a]), str(typ[a]))
    work[nm] = work.get(nm, 0) + (t1[a] - t0[a])
    wait += t0[a] - tq[a]
    if b is not None:
        hop += tq[b] - t1[a]
span = t1.max() - t0.min()
print(json.dumps({"N": N, "n": n, "factor_ms": round(t_f * 1e3, 3), "span_us": round(span / 1e3, 1),
                  "chain_jobs": len(chain), "chain_start_us": round(tq[chain[0]] / 1e3, 1),
                  "work_us": {k: round(v / 1e3, 1) for k, v in sorted(work.items(), key=lambda x: -x[1])},
                  "work_count": {k: sum(1 for a in chain if JT.get(int(typ[a])) == k) for k in work},
                  "enq_to_start_us": round(wait / 1e3, 1), "end_to_enq_us": round(hop / 1e3, 1)}))
if "--list" in sys.argv:
    for a in chain:
        print(f"{JT.get(int(typ[a])):6s} task {int(jt[a, 3] & np.uint64(0xffffffff)):6d} enq {tq[a]/1e3:9.2f} "
              f"start {t0[a]/1e3:9.2f} end {t1[a]/1e3:9.2f} dur {(t1[a]-t0[a])/1e3:7.2f}")
