"""Parity at BASELINE.json's full sizes in the bench's launch configuration (persistent
scheduler, CP priority, nb = 960).  The oracle cannot factor n = 19200 / 46080 in a test,
so: (1) the exact integer family -- L must equal L0 bit for bit; L0 is banded, so the
band is compared and everything else in the lower triangle must be exactly 0;
(2) the uniform family -- sampled entries of A - L L^T obey the componentwise backward
error bound of Cholesky, |A - L L^T|_ij <= gamma_{n+1} (|L| |L|^T)_ij (Higham, Thm 10.3),
computed with torch on the GPU (a checker independent of the library's kernels), and
the diagonal of L is positive."""
import numpy as np
import pytest

import spdgen

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")


def _factor_to_device(n, nb, seed, family):
    import paper_conf_ipps_agullobehkmt15_b200 as c
    with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY) as p:
        c.chol_generate(p.h, seed, family)
        info = c.chol_factor_inplace(p.h)
        L = torch.empty((n, n), dtype=torch.float64, device="cuda")
        c.chol_gather(p.h, L, n)
        torch.cuda.synchronize()
    return L, info


@pytest.mark.parametrize("n", [19200, 46080])
def test_fullsize_integer_family_exact(n):
    nb, seed = 960, 12
    L, info = _factor_to_device(n, nb, seed, 1)
    assert info == 0
    Lb = torch.from_numpy(spdgen.integer_L0_bands(n, seed).astype(np.float64)).cuda()
    idx = torch.arange(n, device="cuda")
    for o in range(spdgen.BW + 1):
        got = L[idx[o:], idx[o:] - o]
        assert torch.equal(got, Lb[o, o:]), o
    # outside the band the exact factor is 0 (lower triangle); upper part must be 0 too
    mask = torch.ones((n, n), dtype=torch.bool, device="cuda")
    for o in range(spdgen.BW + 1):
        mask[idx[o:], idx[o:] - o] = False
    assert int(torch.count_nonzero(L[mask])) == 0
    del L, mask


@pytest.mark.parametrize("n", [19200, 46080])
def test_fullsize_uniform_backward_error_sampled(n):
    nb, seed = 960, 3
    L, info = _factor_to_device(n, nb, seed, 0)
    assert info == 0
    assert bool(torch.all(torch.diagonal(L) > 0))
    assert int(torch.count_nonzero(torch.triu(L[:4096, :4096], 1))) == 0
    rng = np.random.default_rng(n)
    m = 4096
    i = rng.integers(0, n, m)
    j = rng.integers(0, n, m)
    i, j = np.maximum(i, j), np.minimum(i, j)
    i = np.concatenate([i, np.arange(0, n, n // 64)])       # include diagonal entries
    j = np.concatenate([j, np.arange(0, n, n // 64)])
    A = torch.from_numpy(spdgen.uniform_entries(n, seed, i, j)).cuda()
    ti, tj = torch.from_numpy(i).cuda(), torch.from_numpy(j).cuda()
    Li, Lj = L[ti], L[tj]                       # rows i and j (m x n)
    r = A - (Li * Lj).sum(dim=1)
    absdot = (Li.abs() * Lj.abs()).sum(dim=1)
    eps = np.finfo(np.float64).eps
    gamma = (n + 1) * eps / (1 - (n + 1) * eps)
    assert bool(torch.all(r.abs() <= gamma * absdot)), float((r.abs() / (gamma * absdot)).max())
    del L
