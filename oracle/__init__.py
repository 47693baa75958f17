"""ORACLE -- TEST INFRASTRUCTURE ONLY.

Plain CPU reference of the paper's hot path (Agullo et al., HCW 2015,
/root/reference/PAPER.md): the tiled Cholesky factorization of Algorithm 1
(L172-181) and its four tile kernels (L196-208) in ``chol_oracle.c`` (plain C +
OpenMP, fp64, no BLAS), the task graph of Fig. 1 (L213-257) in ``dag.py``, and
the makespan bounds of §III (L334-408, L495-502) in ``bounds.py``.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py`` (its
``cpu_baseline`` leg and ``--impl reference``) may import this package.  It
shares no code with ``paper_conf_ipps_agullobehkmt15_b200`` and never imports it.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "chol_oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")
_lib = None


def build(force: bool = False) -> str:
    """Compile chol_oracle.c -> liboracle.so (gcc -O2 -fopenmp, no -ffast-math)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        cmd = ["gcc", "-O2", "-fopenmp", "-fPIC", "-shared", "-o", _LIB, _SRC, "-lm"]
        subprocess.run(cmd, check=True)
    return _LIB


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_LIB)
        i64, dp, ip = ctypes.c_int64, ctypes.POINTER(ctypes.c_double), ctypes.c_int
        L.oracle_chol_unblocked.argtypes = [i64, dp, i64]
        L.oracle_chol_unblocked.restype = i64
        L.oracle_chol_tiled.argtypes = [i64, i64, dp, i64, ip]
        L.oracle_chol_tiled.restype = i64
        L.oracle_tile_potrf.argtypes = [i64, dp, i64]
        L.oracle_tile_potrf.restype = i64
        L.oracle_tile_trsm.argtypes = [i64, dp, i64, dp, i64]
        L.oracle_tile_trsm.restype = None
        L.oracle_tile_syrk.argtypes = [i64, dp, i64, dp, i64]
        L.oracle_tile_syrk.restype = None
        L.oracle_tile_gemm.argtypes = [i64, dp, i64, dp, i64, dp, i64]
        L.oracle_tile_gemm.restype = None
        L.oracle_chol_solve.argtypes = [i64, dp, i64, dp, i64, i64]
        L.oracle_chol_solve.restype = None
        L.oracle_num_threads.argtypes = [ip]
        L.oracle_num_threads.restype = ip
        _lib = L
    return _lib


def _p(a: np.ndarray):
    assert a.dtype == np.float64 and a.flags.c_contiguous
    return a.ctypes.data_as(ctypes.POINTER(ctypes.c_double))


def chol_unblocked(A: np.ndarray) -> tuple[np.ndarray, int]:
    """Brute-force column Cholesky; returns (L with zeroed upper, info)."""
    L = np.array(A, dtype=np.float64, order="C", copy=True)
    n = L.shape[0]
    info = int(lib().oracle_chol_unblocked(n, _p(L), n))
    if info == 0:
        L[np.triu_indices(n, 1)] = 0.0
    return L, info


def chol_tiled(A: np.ndarray, nb: int, nthreads: int = 0) -> tuple[np.ndarray, int]:
    """Algorithm 1 with tile size nb; returns (L, info) (LAPACK-style info)."""
    L = np.array(A, dtype=np.float64, order="C", copy=True)
    n = L.shape[0]
    info = int(lib().oracle_chol_tiled(n, nb, _p(L), n, nthreads))
    return L, info


def tile_potrf(A: np.ndarray) -> tuple[np.ndarray, int]:
    L = np.array(A, dtype=np.float64, order="C", copy=True)
    nb = L.shape[0]
    info = int(lib().oracle_tile_potrf(nb, _p(L), nb))
    return L, info


def tile_trsm(Lkk: np.ndarray, Aik: np.ndarray) -> np.ndarray:
    Lc = np.ascontiguousarray(Lkk, dtype=np.float64)
    X = np.array(Aik, dtype=np.float64, order="C", copy=True)
    nb = X.shape[0]
    lib().oracle_tile_trsm(nb, _p(Lc), nb, _p(X), nb)
    return X


def tile_syrk(Ljk: np.ndarray, Ajj: np.ndarray) -> np.ndarray:
    Lc = np.ascontiguousarray(Ljk, dtype=np.float64)
    C = np.array(Ajj, dtype=np.float64, order="C", copy=True)
    nb = C.shape[0]
    lib().oracle_tile_syrk(nb, _p(Lc), nb, _p(C), nb)
    return C


def tile_gemm(Lik: np.ndarray, Ljk: np.ndarray, Aij: np.ndarray) -> np.ndarray:
    a = np.ascontiguousarray(Lik, dtype=np.float64)
    b = np.ascontiguousarray(Ljk, dtype=np.float64)
    C = np.array(Aij, dtype=np.float64, order="C", copy=True)
    nb = C.shape[0]
    lib().oracle_tile_gemm(nb, _p(a), nb, _p(b), nb, _p(C), nb)
    return C


def chol_solve(L: np.ndarray, B: np.ndarray) -> np.ndarray:
    """X with L L^T X = B by forward then backward substitution (NEXT-2, L166-171)."""
    Lc = np.ascontiguousarray(L, dtype=np.float64)
    X = np.array(B, dtype=np.float64, order="C", copy=True)
    if X.ndim == 1:
        X = X.reshape(-1, 1)
    n, nrhs = X.shape
    lib().oracle_chol_solve(n, _p(Lc), n, _p(X), nrhs, nrhs)
    return X.reshape(B.shape)


def num_threads(nthreads: int = 0) -> int:
    return int(lib().oracle_num_threads(nthreads))


def flops(n: int) -> float:
    """Leading-order flop count n^3/3 the metric uses (BASELINE.json, reading R7)."""
    return n ** 3 / 3.0


def flops_exact(n: int) -> float:
    """LAPACK dpotrf count n^3/3 + n^2/2 + n/6 (reading R7)."""
    return n ** 3 / 3.0 + n ** 2 / 2.0 + n / 6.0


def backward_error(A: np.ndarray, L: np.ndarray) -> float:
    """||A - L L^T||_F / (n eps ||A||_F) using the lower triangle of A (symmetrised)."""
    n = A.shape[0]
    As = np.tril(A) + np.tril(A, -1).T
    R = As - L @ L.T
    return float(np.linalg.norm(R) / (n * np.finfo(np.float64).eps * np.linalg.norm(As)))


def rel_diff(L: np.ndarray, Lref: np.ndarray) -> dict:
    """Elementwise difference on the lower triangle (reading R8): floored max
    relative difference, unfloored max, and Frobenius relative difference."""
    tri = np.tril_indices(L.shape[0])
    a, b = L[tri], Lref[tri]
    scale = np.max(np.abs(b)) if b.size else 1.0
    floor = np.maximum(np.abs(b), 1e-6 * scale)
    d = np.abs(a - b)
    with np.errstate(divide="ignore", invalid="ignore"):
        unf = np.where(b != 0, d / np.abs(b), np.where(d == 0, 0.0, np.inf))
    return {"max_rel_floored": float(np.max(d / floor)) if d.size else 0.0,
            "max_rel": float(np.max(unf)) if d.size else 0.0,
            "fro_rel": float(np.linalg.norm(d) / max(np.linalg.norm(b), 1e-300))}
