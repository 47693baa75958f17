import sys, numpy as np, torch
sys.path.insert(0, '.')
import numpy as np
import spdgen  # reference: LAPACK through numpy (the oracle is test infrastructure only)
import paper_conf_ipps_agullobehkmt15_b200 as c
for nb in [192, 288, 960]:
    n = 3 * nb
    M = spdgen.uniform_spd(n, seed=21)
    with c.Plan(n, nb, executor=c.EXEC_HOST) as p:
        dM = torch.from_numpy(M).cuda()
        c.chol_scatter(p.h, dM, n)
        c.chol_run_task(p.h, 0, 1, 1, 1, 1)
        out = torch.empty_like(dM); c.chol_gather(p.h, out, n); torch.cuda.synchronize()
        out = out.cpu().numpy()
    T = out[nb:2*nb, nb:2*nb]
    ref, info = np.linalg.cholesky(M[nb:2*nb, nb:2*nb]), 0
    ref = np.tril(ref); T = np.tril(T)
    err = np.abs(T - ref) / np.maximum(np.abs(ref), 1e-6 * np.abs(ref).max())
    bad = np.argwhere(err > 1e-12)
    print("nb", nb, "nbad", len(bad), "max", err.max())
    if len(bad):
        cols = bad[:, 1]; rows = bad[:, 0]
        j = cols.min(); print(" first bad col", j, "rows in that col", rows[cols == j][:20], "block", j // 96)
        # error by block
        BS = 96
        for bi in range(nb // BS):
            for bj in range(bi + 1):
                e = err[bi*BS:(bi+1)*BS, bj*BS:(bj+1)*BS].max()
                if e > 1e-12: print("  block", bi, bj, "%.3e" % e)
