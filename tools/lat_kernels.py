import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_agullobehkmt15_b200 as c
nb = 960
with c.Plan(3 * nb, nb, executor=c.EXEC_HOST) as p:
    c.chol_generate(p.h, 1, 0)
    for t in (0, 1):
        c.chol_run_task(p.h, t, 2, 1, 0 if t else 1, 1)
