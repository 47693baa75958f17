"""Policy ablation (BASELINE configs[4]): DYNAMIC vs CP_PRIORITY vs STATIC with a sweep of
the TRSM pin distance d and of the latency-worker count."""
import sys, os, json
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c

n = int(sys.argv[1]) if len(sys.argv) > 1 else 28800
nb = 960
N = n // nb
reps = 3


def run(**opts):
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, **opts) as p:
        ts = []
        for r in range(reps + 1):
            c.chol_generate(p.h, 0, 0)
            assert c.chol_factor_inplace(p.h) == 0
            if r:
                ts.append(c.chol_last_times(p.h)[0])
    t = min(ts)
    return {"opts": opts, "ms": round(t * 1e3, 3), "tflops": round(n ** 3 / 3 / t / 1e12, 3)}


out = [run(policy=c.POLICY_DYNAMIC), run(policy=c.POLICY_CP_PRIORITY)]
for lw in (8, 16, 32):
    for d in (1, 2, 4, 8, N - 1):
        out.append(run(policy=c.POLICY_STATIC, trsm_pin_distance=d, latency_workers=lw))
for o in out:
    print(json.dumps({"n": n, **o}))
