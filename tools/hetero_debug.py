"""Step-by-step replay of tests/test_gpu_production.py::test_host_cpu_class_trsms_match_oracle
(without the oracle) with progress prints, to locate a stall."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import paper_conf_ipps_agullobehkmt15_b200 as c
import spdgen

N, d = int(sys.argv[1]), int(sys.argv[2])
nb = 960
n = N * nb
A = spdgen.uniform_spd(n, N + 100)
print("plan", flush=True)
with c.Plan(n, nb, cpu_trsm_distance=d) as p:
    dA = torch.from_numpy(A).cuda()
    t = time.time(); print("factor device", p.factor(dA), time.time() - t, flush=True)
    L = np.full_like(A, np.nan)
    t = time.time(); print("factor host", c.chol_factor(p.h, A, n, L, n), time.time() - t, flush=True)
    c.chol_generate(p.h, 4, 1)
    t = time.time(); print("factor inplace", c.chol_factor_inplace(p.h), time.time() - t, flush=True)
print("done", flush=True)
