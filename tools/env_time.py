"""A/B of development switches: factorization time per environment setting, per n
(nb = 960, CP priority, best and median of 5 after 2 warm-ups), with a bitwise check of
the factor against the default setting's (R15: the schedule never changes the bits).

  python tools/env_time.py 9600,19200 "" "CHOL_BLOCK_HEAD=1" "CHOL_BLOCK_HEAD=1 CHOL_BLOCK_TAIL=3"
"""
import json, os, statistics, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
import paper_conf_ipps_agullobehkmt15_b200 as c

Ns = [int(x) for x in sys.argv[1].split(",")]
sets = sys.argv[2:] or [""]
nb = 960
for n in Ns:
    ref = None
    for s in sets:
        env = dict(kv.split("=") for kv in s.split()) if s else {}
        old = {k: os.environ.get(k) for k in env}
        os.environ.update(env)
        with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
            ts = []
            for r in range(7):
                c.chol_generate(p.h, 0, 0)
                assert c.chol_factor_inplace(p.h) == 0
                if r >= 2:
                    ts.append(c.chol_last_times(p.h)[0])
            L = torch.empty(n, n, dtype=torch.float64, device="cuda")
            c.chol_gather(p.h, L.data_ptr(), n)
        for k, v in old.items():
            if v is None:
                os.environ.pop(k, None)
            else:
                os.environ[k] = v
        same = None
        if ref is None:
            ref = L
        else:
            same = bool(torch.equal(ref, L))
        print(json.dumps({"n": n, "env": s, "best_ms": round(min(ts) * 1e3, 3),
                          "median_ms": round(statistics.median(ts) * 1e3, 3),
                          "tflops_best": round(n ** 3 / 3 / min(ts) / 1e12, 2), "bitwise_equal_to_first": same}),
              flush=True)
        del L
        torch.cuda.empty_cache()
