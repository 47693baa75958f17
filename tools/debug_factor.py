import sys, os, numpy as np, torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import spdgen  # the oracle is test infrastructure only: LAPACK (numpy) is the reference here
import paper_conf_ipps_agullobehkmt15_b200 as c
n, nb = int(sys.argv[1]), int(sys.argv[2])
ex = int(sys.argv[3]) if len(sys.argv) > 3 else 1
A = spdgen.uniform_spd(n, seed=n + nb)
ref = np.linalg.cholesky(A)
BS = 96 if nb % 96 == 0 else 64 if nb % 64 == 0 else 32
outs = []
for rep in range(6):
    with c.Plan(n, nb, executor=ex) as p:
        dA = torch.from_numpy(A.copy()).cuda()
        info = p.factor(dA); torch.cuda.synchronize()
        L = dA.cpu().numpy()
    outs.append(L)
    err = np.abs(L - ref) / np.maximum(np.abs(ref), 1e-6 * np.abs(ref).max())
    bad = np.argwhere(np.tril(err) > 1e-10)
    blocks = sorted(set((int(a) // BS, int(b) // BS) for a, b in bad))
    print("rep", rep, "info", info, "max", err.max(), "nbad", len(bad), "first bad blocks", blocks[:12],
          "same as rep0", np.array_equal(L, outs[0]))
    if len(bad):
        j = bad[:, 1].min()
        print("   first bad col", j, "rows", bad[bad[:, 1] == j][:10, 0])
