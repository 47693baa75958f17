"""Hybrid-DAG sweep: factorization time vs the number m of trailing steps built at block
granularity (CHOL_BLOCK_TAIL), per N (nb = 960, CP priority, best of 3 after a warm-up)."""
import json, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c
Ns = [int(x) for x in sys.argv[1].split(",")]
ms = [int(x) for x in sys.argv[2].split(",")]
nb = 960
for N in Ns:
    n = N * nb
    row = {"N": N}
    for m in ms:
        if m > N:
            continue
        os.environ["CHOL_BLOCK_TAIL"] = str(m)
        with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
            ts = []
            for r in range(4):
                c.chol_generate(p.h, 0, 0)
                assert c.chol_factor_inplace(p.h) == 0
                if r:
                    ts.append(c.chol_last_times(p.h)[0])
        row[f"m{m}"] = round(min(ts) * 1e3, 3)
    print(json.dumps(row), flush=True)
