"""STATIC-policy sweep at one n: latency workers x pin distance x TRSM decomposition of the
pinned TRSMs (env CHOL_TRSM_DIST / CHOL_TRSM_SLABCHAIN set by the caller)."""
import json, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c

n = int(sys.argv[1]) if len(sys.argv) > 1 else 9600
lws = [int(x) for x in sys.argv[2].split(",")] if len(sys.argv) > 2 else [16, 32]
ds = [int(x) for x in sys.argv[3].split(",")] if len(sys.argv) > 3 else [1, 2]
nb = 960


def run(**opts):
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, **opts) as p:
        ts = []
        for r in range(4):
            c.chol_generate(p.h, 0, 0)
            assert c.chol_factor_inplace(p.h) == 0
            if r:
                ts.append(c.chol_last_times(p.h)[0])
    t = min(ts)
    return {"env": {k: v for k, v in os.environ.items() if k.startswith("CHOL_")}, "opts": opts, "n": n,
            "ms": round(t * 1e3, 3), "tflops": round(n ** 3 / 3 / t / 1e12, 3)}


print(json.dumps(run(policy=c.POLICY_CP_PRIORITY)), flush=True)
for lw in lws:
    for d in ds:
        print(json.dumps(run(policy=c.POLICY_STATIC, trsm_pin_distance=d, latency_workers=lw)), flush=True)
