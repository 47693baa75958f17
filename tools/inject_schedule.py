"""NEXT-4 on the device: the exact task-level schedule of a small factorization (a one-class
model of the GPU: W task slots, each task taking its measured T_lat -- a GEMM alone fills
~100 of the 148 SMs, so about two tasks run side by side) injected into the persistent
scheduler as static priorities (minus the start rank), against the default bottom-level
priorities and DYNAMIC.  Prints one JSON line per N.
  python tools/inject_schedule.py 4,5,6 [slots]"""
import json, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import paper_conf_ipps_agullobehkmt15_b200 as c

Ns = [int(x) for x in sys.argv[1].split(",")] if len(sys.argv) > 1 else [4, 5, 6]
slots = int(sys.argv[2]) if len(sys.argv) > 2 else 2
nb = 960


def best_of(p, reps=7):
    ts, L = [], None
    for r in range(reps):
        c.chol_generate(p.h, 0, 0)
        assert c.chol_factor_inplace(p.h) == 0
        ts.append(c.chol_last_times(p.h)[0])
    out = torch.empty((p.n, p.n), dtype=torch.float64, device="cuda")
    c.chol_gather(p.h, out, p.n)
    return min(ts[1:]), out


for N in Ns:
    n = N * nb
    with c.Plan(n, nb) as p:
        c.chol_generate(p.h, 0, 0)
        T_lat = [c.chol_run_batch(p.h, t, 1, 5) * 1e-3 for t in range(4)]
    mk, optimal, w, r, nodes = c.chol_optimal_schedule(N, [slots], [T_lat], node_limit=20_000_000)
    res = {"N": N, "n": n, "model": {"slots": slots, "T_lat_us": [round(x * 1e6, 1) for x in T_lat],
                                     "optimal_makespan_ms": mk * 1e3, "proven": optimal, "nodes": nodes}}
    with c.Plan(n, nb) as p:
        t_cp, L_cp = best_of(p)
    with c.Plan(n, nb, policy=c.POLICY_DYNAMIC) as p:
        t_dyn, _ = best_of(p)
    with c.Plan(n, nb) as p:
        c.chol_set_task_priorities(p.h, [-x for x in r])
        t_inj, L_inj = best_of(p)
    res.update({"cp_ms": t_cp * 1e3, "dynamic_ms": t_dyn * 1e3, "injected_ms": t_inj * 1e3,
                "bitwise_equal": bool(torch.equal(L_cp, L_inj))})
    print(json.dumps(res), flush=True)
