import sys, numpy as np, torch
sys.path.insert(0, '.')
import spdgen
import paper_conf_ipps_agullobehkmt15_b200 as c
def run(nb, typ, reps=1):
    n = 3 * nb
    M = spdgen.uniform_spd(n, seed=24)
    outs = []
    for r in range(2):
        with c.Plan(n, nb, executor=c.EXEC_HOST) as p:
            dM = torch.from_numpy(M).cuda()
            c.chol_scatter(p.h, dM, n)
            if typ == 3: c.chol_run_task(p.h, 3, 2, 1, 0, 1)
            else: c.chol_run_task(p.h, 2, 1, 1, 0, 1)
            out = torch.empty_like(dM); c.chol_gather(p.h, out, n); torch.cuda.synchronize()
            outs.append(out.cpu().numpy())
    T = lambda X, i, j: X[i*nb:(i+1)*nb, j*nb:(j+1)*nb]
    if typ == 3:
        ref = T(M,2,1) - T(M,2,0) @ T(M,1,0).T; got = T(outs[0],2,1); got2 = T(outs[1],2,1)
    else:
        ref = np.tril(T(M,1,1) - T(M,1,0) @ T(M,1,0).T); got = np.tril(T(outs[0],1,1)); got2 = np.tril(T(outs[1],1,1))
    err = np.abs(got - ref)
    print("nb", nb, "type", typ, "max abs err", err.max(), "runs identical", np.array_equal(got, got2))
    BS = 96 if nb % 96 == 0 else 64 if nb % 64 == 0 else 32
    if err.max() > 1e-9:
        bad = np.argwhere(err > 1e-9)
        print("  nbad", len(bad), "rows mod BS", np.unique(bad[:,0] % BS)[:50], "cols mod BS", np.unique(bad[:,1] % BS)[:50])
        print("  blocks", sorted(set((int(a)//BS, int(b)//BS) for a, b in bad))[:20])
for nb in [64, 128, 192, 256, 96]:
    for typ in (3, 2):
        run(nb, typ)
