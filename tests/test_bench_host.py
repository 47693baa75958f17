"""Host logic of bench.py (no GPU): the multi-GPU workload rule and the process grid."""
import types

import bench


def _args(**kw):
    a = dict(n=19200, nb=960, scaling="weak", grid="")
    a.update(kw)
    return types.SimpleNamespace(**a)


def test_weak_scaling_keeps_flops_per_gpu():
    a = _args()
    ns = {ws: bench.workload_n(a, ws) for ws in (1, 2, 4, 8)}
    assert ns == {1: 19200, 2: 24000, 4: 30720, 8: 38400}
    per_gpu = [n ** 3 / 3 / ws for ws, n in ns.items()]
    assert max(per_gpu) / min(per_gpu) < 1.06  # within the rounding of n to whole tiles
    assert all(n % 960 == 0 for n in ns.values())


def test_strong_scaling_keeps_n():
    a = _args(scaling="strong")
    assert {bench.workload_n(a, ws) for ws in (1, 2, 4, 8)} == {19200}


def test_grid_prefers_p_le_q():
    a = _args()
    assert bench.grid_of(a, 2) == (1, 2)
    assert bench.grid_of(a, 4) == (2, 2)
    assert bench.grid_of(a, 8) == (2, 4)
    assert bench.grid_of(_args(grid="1x8"), 8) == (1, 8)
