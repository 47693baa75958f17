"""Sweep-level trace of chol_solve (development; CHOL_SOLVE_TRACE): per block row b, when
its item was claimed, when its chain stage began waiting for block row b-1 and saw it,
when b was published.  Splits the step time t_pub(b) - t_pub(b-1) into
  late  = max(0, t_chainwait(b) - t_pub(b-1))   item b not yet at its chain stage
  hop   = t_seen(b) - max(t_chainwait(b), t_pub(b-1))   flag propagation
  tail  = t_pub(b) - t_seen(b)                   fetch Y_{b-1}, chain FMA, store, publish"""
import json, os, sys, tempfile
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
n = int(sys.argv[1]) if len(sys.argv) > 1 else 19200
nrhs = int(sys.argv[2]) if len(sys.argv) > 2 else 1
path = os.path.join(tempfile.mkdtemp(), "solve_trace.bin")
import paper_conf_ipps_agullobehkmt15_b200 as c
import spdgen
with c.Plan(n, 960) as p:
    c.chol_generate(p.h, 0, 0)
    assert c.chol_factor_inplace(p.h) == 0
    B0 = spdgen.rhs(n, nrhs, 1)
    for r in range(3):
        B = B0.copy()
        c.chol_solve(p.h, B, nrhs, nrhs)
    sw = c.chol_last_solve_times(p.h)[1]
    os.environ["CHOL_SOLVE_TRACE"] = path
    B = B0.copy()
    c.chol_solve(p.h, B, nrhs, nrhs)
    del os.environ["CHOL_SOLVE_TRACE"]
t = np.fromfile(path, dtype=np.uint64).reshape(-1, 6).astype(np.int64)
half = len(t) // 2
out = {"n": n, "nrhs": nrhs, "sweeps_ms_untraced": round(sw * 1e3, 4)}
for name, tt in (("forward", t[:half]), ("backward", t[half:])):
    b = tt[:, 5] >> 32
    o = np.argsort(b) if name == "forward" else np.argsort(-b)
    tt = tt[o]
    t0 = tt[:, 0].min()
    claim, cw, cs, pub, wait = (tt[:, k] - (t0 if k < 4 else 0) for k in range(5))
    step = np.diff(pub)
    late = np.maximum(0, cw[1:] - pub[:-1])
    hop = cs[1:] - np.maximum(cw[1:], pub[:-1])
    tail = pub[1:] - cs[1:]
    m = len(step)
    q = [0, m // 4, m // 2, 3 * m // 4, m]
    out[name] = {"span_us": round((pub.max()) / 1e3, 1), "steps": m,
                 "step_us_by_quarter": [round(float(step[q[i]:q[i + 1]].mean()) / 1e3, 2) for i in range(4)],
                 "late_us_by_quarter": [round(float(late[q[i]:q[i + 1]].mean()) / 1e3, 2) for i in range(4)],
                 "hop_us_mean": round(float(hop.mean()) / 1e3, 2), "tail_us_mean": round(float(tail.mean()) / 1e3, 2),
                 "item_us_by_quarter": [round(float((pub - claim)[q[i]:q[i + 1]].mean()) / 1e3, 1) for i in range(4)],
                 "older_wait_us_mean": round(float(wait.mean()) / 1e3, 1)}
print(json.dumps(out))
