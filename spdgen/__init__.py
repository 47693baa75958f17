"""Seeded synthetic SPD inputs shared by the oracle side and the CUDA side.

This module holds NO Cholesky arithmetic: it only draws the matrices the paper's
method is applied to (the paper factors "a dense, symmetric, and positive-definite
double-precision matrix A", in tiles of nb=960, L690-693).
The recipe is stated in DESIGN.md §"Input recipe"; it is counter based
(splitmix64 of the element index), so the CUDA library's own device generator
(`chol_generate`) implements the same function independently and a test checks
the two bit for bit.

Families
--------
* ``uniform``: A[i][j] = u(i,j) + n*[i==j], u in [-0.5, 0.5) from the hash of
  (seed, max(i,j), min(i,j)).  Symmetric by construction; Gershgorin gives a
  diagonal excess >= n/2, so A is SPD with condition number <~ 3.
* ``integer``: A = L0 L0^T with L0 lower triangular, banded (bandwidth BW=3),
  off-diagonals in {-1, 0, +1}, diagonal in {1, 2, 4}.  Every quantity a
  Cholesky factorization computes on it is an integer far below 2^53 (divisions
  are by 1, 2 or 4), so any correct algorithm, in any summation order, returns
  exactly L0.
"""
from __future__ import annotations

import numpy as np

GOLDEN = np.uint64(0x9E3779B97F4A7C15)
M1 = np.uint64(0xBF58476D1CE4E5B9)
M2 = np.uint64(0x94D049BB133111EB)
INT_SALT = np.uint64(0xD1B54A32D192ED03)  # separates the integer family's stream
BW = 3  # bandwidth of L0 in the integer family

__all__ = ["splitmix64", "uniform_spd", "uniform_entries", "integer_L0", "integer_L0_bands", "integer_spd",
           "make_non_spd", "BW", "rhs", "integer_rhs_solution"]


def splitmix64(x: np.ndarray) -> np.ndarray:
    """splitmix64 finaliser of x + golden (all arithmetic mod 2^64)."""
    with np.errstate(over="ignore"):
        z = x.astype(np.uint64, copy=True)
        z += GOLDEN
        z = (z ^ (z >> np.uint64(30))) * M1
        z = (z ^ (z >> np.uint64(27))) * M2
        z ^= z >> np.uint64(31)
    return z


def _u01(z: np.ndarray) -> np.ndarray:
    """Top 53 bits as a double in [0,1) -- exact in FP64."""
    return (z >> np.uint64(11)).astype(np.float64) * (2.0 ** -53)


def uniform_spd(n: int, seed: int = 0, *, rows: slice | None = None,
                upper: str = "mirror") -> np.ndarray:
    """The ``uniform`` family, row-major (n x n) float64.

    ``upper``: "mirror" fills the full symmetric matrix; "nan" fills the
    strictly upper triangle with NaN (the factorization must read only the
    lower triangle); "zero" with zeros.
    """
    r0, r1 = (0, n) if rows is None else (rows.start or 0, rows.stop or n)
    out = np.empty((r1 - r0, n), dtype=np.float64)
    with np.errstate(over="ignore"):
        base = np.uint64(seed) * GOLDEN
        j = np.arange(n, dtype=np.uint64)
        step = 512
        for a in range(r0, r1, step):
            b = min(a + step, r1)
            i = np.arange(a, b, dtype=np.uint64)[:, None]
            hi = np.maximum(i, j[None, :])
            lo = np.minimum(i, j[None, :])
            key = base + hi * np.uint64(n) + lo
            blk = _u01(splitmix64(key)) - 0.5
            ii = np.arange(a, b)
            sel = (ii >= 0) & (ii < n)
            blk[np.arange(b - a)[sel], ii[sel]] += float(n)
            if upper != "mirror":
                mask = np.arange(n)[None, :] > ii[:, None]
                blk[mask] = np.nan if upper == "nan" else 0.0
            out[a - r0:b - r0] = blk
    return out


def uniform_entries(n: int, seed: int, i: np.ndarray, j: np.ndarray) -> np.ndarray:
    """Entries A[i, j] of the ``uniform`` family for index arrays (any size n)."""
    i = np.asarray(i, dtype=np.uint64)
    j = np.asarray(j, dtype=np.uint64)
    with np.errstate(over="ignore"):
        key = np.uint64(seed) * GOLDEN + np.maximum(i, j) * np.uint64(n) + np.minimum(i, j)
    v = _u01(splitmix64(key)) - 0.5
    return np.where(i == j, v + float(n), v)


def _int_hash(n: int, seed: int, i: np.ndarray, j: np.ndarray) -> np.ndarray:
    with np.errstate(over="ignore"):
        key = (np.uint64(seed) ^ INT_SALT) * GOLDEN + i.astype(np.uint64) * np.uint64(n) \
            + j.astype(np.uint64)
    return splitmix64(key)


def integer_L0_bands(n: int, seed: int = 0) -> np.ndarray:
    """Bands of L0: ``Lb[o, i] = L0[i, i-o]`` for o = 0..BW (0 where i-o < 0)."""
    Lb = np.zeros((BW + 1, n), dtype=np.int64)
    i = np.arange(n)
    zd = _int_hash(n, seed, i, i)
    Lb[0] = np.array([1, 2, 4], dtype=np.int64)[((zd >> np.uint64(32)) % np.uint64(3)).astype(np.int64)]
    for o in range(1, BW + 1):
        ii = i[o:]
        z = _int_hash(n, seed, ii, ii - o)
        top = (z >> np.uint64(61)).astype(np.int64)  # 0..7
        v = np.where(top < 2, -1, np.where(top < 4, 1, 0))
        Lb[o, o:] = v
    return Lb


def integer_L0(n: int, seed: int = 0) -> np.ndarray:
    """Dense L0 (float64, row-major) of the ``integer`` family."""
    Lb = integer_L0_bands(n, seed)
    L = np.zeros((n, n), dtype=np.float64)
    i = np.arange(n)
    for o in range(BW + 1):
        L[i[o:], i[o:] - o] = Lb[o, o:]
    return L


def integer_spd(n: int, seed: int = 0, *, upper: str = "mirror") -> np.ndarray:
    """A = L0 L0^T of the ``integer`` family, computed exactly in int64 from the bands."""
    Lb = integer_L0_bands(n, seed)
    A = np.zeros((n, n), dtype=np.float64)
    i = np.arange(n)
    # A[i, i-o] = sum_{p=o..BW} L0[i, i-p] * L0[i-o, i-p] = sum_p Lb[p, i] * Lb[p-o, i-o]
    for o in range(BW + 1):
        acc = np.zeros(n - o, dtype=np.int64)
        for p in range(o, BW + 1):
            acc += Lb[p, o:] * Lb[p - o, :n - o]
        A[i[o:], i[o:] - o] = acc
        if upper == "mirror":
            A[i[o:] - o, i[o:]] = acc
    if upper == "nan":
        A[np.triu_indices(n, 1)] = np.nan
    return A


def make_non_spd(A: np.ndarray, L0: np.ndarray, j0: int, kind: str = "zero") -> np.ndarray:
    """Integer family made non-SPD at column j0 (0-based).

    kind="zero": subtract L0[j0,j0]^2 from A[j0,j0] -> the pivot at j0 is exactly 0.
    kind="neg":  subtract L0[j0,j0]^2 + 1 -> the pivot is exactly -1.
    In both cases a correct factorization reports info = j0 + 1 (LAPACK convention).
    """
    B = A.copy()
    d = L0[j0, j0] ** 2 + (1.0 if kind == "neg" else 0.0)
    B[j0, j0] -= d
    return B


RHS_SALT = np.uint64(0x5851F42D4C957F2D)


def rhs(n: int, nrhs: int, seed: int = 0) -> np.ndarray:
    """Right-hand sides for the solve: n x nrhs row-major, entries
    u in [-0.5, 0.5) from splitmix64 of (seed ^ RHS_SALT, row, column)."""
    i = np.arange(n, dtype=np.uint64)[:, None]
    j = np.arange(nrhs, dtype=np.uint64)[None, :]
    with np.errstate(over="ignore"):
        key = (np.uint64(seed) ^ RHS_SALT) * GOLDEN + i * np.uint64(nrhs) + j
    return _u01(splitmix64(key)) - 0.5


def integer_rhs_solution(n: int, nrhs: int, seed: int = 0) -> np.ndarray:
    """Small integer solutions X0 in {-2..2} (n x nrhs): with the integer family, B = A X0
    is an exact integer matrix and the substitutions return X0 exactly."""
    i = np.arange(n, dtype=np.uint64)[:, None]
    j = np.arange(nrhs, dtype=np.uint64)[None, :]
    with np.errstate(over="ignore"):
        key = (np.uint64(seed) ^ RHS_SALT ^ INT_SALT) * GOLDEN + i * np.uint64(nrhs) + j
    return ((splitmix64(key) >> np.uint64(61)).astype(np.int64) % 5 - 2).astype(np.float64)
