"""CPU-only checks of the C-ABI library: it builds, loads without a GPU, exports every
symbol include/chol.h declares, and its host-side rows of the hot path -- the task
graph and the bounds (A9) -- agree with the oracle."""
import ctypes
import os
import re

import pytest

from oracle import bounds as obounds
from oracle import dag as odag

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def chol():
    from paper_conf_ipps_agullobehkmt15_b200 import build
    build.build()
    import paper_conf_ipps_agullobehkmt15_b200 as c
    return c


def declared_symbols():
    src = open(os.path.join(ROOT, "include", "chol.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(chol_[a-z_]+)\s*\(", src)))


def test_header_symbols_exported(chol):
    lib = ctypes.CDLL(chol.LIB_PATH)
    syms = declared_symbols()
    assert len(syms) >= 19
    for s in syms:
        assert hasattr(lib, s), s
    assert set(syms) == set(chol.EXPORTED)


def test_strerror(chol):
    assert chol.chol_strerror(0) == "success"
    assert "n <= 0" in chol.chol_strerror(-1)


def test_no_gpu_plan_fails_loudly(chol):
    import torch
    if torch.cuda.is_available():
        pytest.skip("GPU present")
    with pytest.raises(chol.CholError) as e:
        chol.chol_plan(1024, 256)
    assert e.value.status == -3


@pytest.mark.parametrize("N", [1, 2, 3, 5, 8, 12])
def test_dag_matches_oracle(chol, N):
    nt, E = chol.chol_dag(N)
    ts, OE = odag.edges(N)
    assert nt == len(ts)
    ids = [chol.chol_task_id(N, t.type, t.i, t.j, t.k) for t in ts]
    assert sorted(ids) == list(range(nt))
    oracle_edges = {(ids[p], ids[s]) for p, s in OE}
    assert set(E) == oracle_edges and len(E) == len(OE)


def test_bounds_match_oracle(chol):
    T_lat = [5e-4, 2e-4, 9e-5, 9e-5]
    T_thr = [1.2e-4, 1.1e-4, 3.6e-5, 5.7e-5]
    keys = ["POTRF", "TRSM", "SYRK", "GEMM"]
    for n, nb, M in [(9600, 960, 1), (19200, 960, 1), (46080, 960, 8), (1024, 256, 2)]:
        got = chol.chol_bounds(n, nb, M, T_lat, T_thr)
        ref = obounds.all_bounds(n, nb, dict(zip(keys, T_thr)), dict(zip(keys, T_lat)), M)
        for k in ("area", "chain", "mixed", "critical_path", "gemm_peak"):
            assert abs(got[k] - ref[k]) <= 1e-12 * max(1.0, abs(ref[k])), (k, got[k], ref[k])


def test_owner_area_matches_oracle(chol):
    keys = ["POTRF", "TRSM", "SYRK", "GEMM"]
    T_thr = [1.2e-4, 1.1e-4, 3.6e-5, 5.7e-5]
    for N, p, q in [(1, 1, 1), (7, 1, 2), (20, 2, 2), (25, 1, 2), (40, 2, 4), (48, 4, 2), (13, 3, 3)]:
        mx, per = chol.chol_owner_area(N, p, q, T_thr)
        rmx, rper = obounds.owner_area(N, p, q, dict(zip(keys, T_thr)))
        assert abs(mx - rmx) <= 1e-12 * rmx
        assert all(abs(a - b) <= 1e-12 * max(b, 1e-30) for a, b in zip(per, rper))


@pytest.mark.parametrize("nb,bs", [(96, 96), (192, 96), (960, 96), (128, 64), (64, 32)])
def test_cpu_class_trsm_kernel_matches_oracle(nb, bs, chol):
    """NEXT-3: the host CPU class's tile TRSM (inverse form, AVX-512 dot-product kernel)
    against the oracle's substitution, and exact on the integer family (R19)."""
    import numpy as np
    import oracle
    import spdgen
    c = chol
    M = spdgen.uniform_spd(2 * nb, nb + bs)
    L = np.ascontiguousarray(np.linalg.cholesky(M[:nb, :nb]))
    X = np.ascontiguousarray(M[nb:, :nb])
    ref = oracle.tile_trsm(L, X)
    got = X.copy()
    c.chol_cpu_trsm(got, L, bs)
    scale = np.max(np.abs(ref))
    assert np.max(np.abs(got - ref) / np.maximum(np.abs(ref), 1e-6 * scale)) <= 1e-10
    L0 = spdgen.integer_L0(2 * nb, 7)
    A = spdgen.integer_spd(2 * nb, 7)
    Xi = np.ascontiguousarray(A[nb:, :nb])
    c.chol_cpu_trsm(Xi, np.ascontiguousarray(L0[:nb, :nb]), bs)
    assert np.array_equal(Xi, L0[nb:, :nb])
    with pytest.raises(c.CholError):
        c.chol_cpu_trsm(X.copy(), L, 7)
