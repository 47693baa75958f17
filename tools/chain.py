"""Critical-chain timeline from the task trace: POTRF_k, TRSM_{k+1,k}, SYRK_{k+1,k}."""
import sys, os, json
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c
n = int(sys.argv[1]) if len(sys.argv) > 1 else 19200
pol = int(sys.argv[2]) if len(sys.argv) > 2 else 0  # 0 = CP_PRIORITY
nb = 960
with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=pol, trace=1) as p:
    for rep in range(2):
        c.chol_generate(p.h, 0, 0)
        c.chol_factor_inplace(p.h)
    recs, mk = c.chol_trace(p.h)
N = n // nb
idx = {(r["type"], r["i"], r["j"], r["k"]): r for r in recs}
print("makespan_ms", round(mk * 1e3, 2))
for k in list(range(0, 6)) + list(range(N - 4, N)):
    P = idx[(0, k, k, k)]
    line = f"k={k:2d} POTRF {P['t0_ns']/1e3:9.1f}-{P['t1_ns']/1e3:9.1f}"
    if k + 1 < N:
        T = idx[(1, k + 1, k, k)]
        S = idx[(2, k + 1, k + 1, k)]
        Tall = [idx[(1, i, k, k)] for i in range(k + 1, N)]
        line += f" | TRSM_{k+1} {T['t0_ns']/1e3:9.1f}-{T['t1_ns']/1e3:9.1f} (all TRSM done {max(r['t1_ns'] for r in Tall)/1e3:9.1f})"
        line += f" | SYRK {S['t0_ns']/1e3:9.1f}-{S['t1_ns']/1e3:9.1f}"
    print(line)
