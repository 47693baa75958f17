"""ORACLE -- TEST INFRASTRUCTURE ONLY.  Makespan lower bounds of PAPER.md §III.

Reading R9-R12: with one resource type (the GPU, M = number of
GPUs), the area LP (L349-359) has the closed form area = sum_t N_t T_t / M
(LP relaxation, reading R10); the mixed bound adds the chain constraint
(L388-396)  N T_P + (N-1) T*_T + (N-1) T*_S <= l, so mixed = max(area, chain);
the critical-path bound (L495-498) is the longest DAG path with each task's
fastest time; the GEMM-peak bound (L122-134, L499-502) is total flops over the
aggregate GEMM rate.  Area terms use throughput times T_thr (a saturated GPU),
path terms use latency times T_lat (a task alone), reading R9.

The general R-resource-type LP (several resource classes) is solved with
scipy's linprog (LP relaxation of n_rt in N+).
"""
from __future__ import annotations

from . import dag


def task_counts(N: int) -> dict[str, int]:
    """Closed forms N_P=N, N_T=N_S=N(N-1)/2, N_G=N(N-1)(N-2)/6 (text L383-386)."""
    return {"POTRF": N, "TRSM": N * (N - 1) // 2, "SYRK": N * (N - 1) // 2,
            "GEMM": N * (N - 1) * (N - 2) // 6}


def area(N: int, T_thr: dict[str, float], M: int = 1) -> float:
    c = task_counts(N)
    return sum(c[t] * T_thr[t] for t in c) / M


def chain(N: int, T_lat: dict[str, float]) -> float:
    """The diagonal path of all N POTRFs, N-1 TRSMs and N-1 SYRKs (L383-396)."""
    return N * T_lat["POTRF"] + (N - 1) * (T_lat["TRSM"] + T_lat["SYRK"])


def mixed(N: int, T_thr: dict[str, float], T_lat: dict[str, float], M: int = 1) -> float:
    return max(area(N, T_thr, M), chain(N, T_lat))


def critical_path(N: int, T_lat: dict[str, float]) -> float:
    """Longest path of the brute-force DAG with task weight T_lat[type] (L495-498)."""
    return dag.longest_path(N, lambda t: T_lat[dag.TYPE_NAMES[t.type]])


def gemm_peak(n: int, nb: int, T_G_thr: float, M: int = 1) -> float:
    """(n^3/3) / (M * R_G) with R_G = 2 nb^3 / T_G (L499-502)."""
    R_G = 2.0 * nb ** 3 / T_G_thr
    return (n ** 3 / 3.0) / (M * R_G)


def all_bounds(n: int, nb: int, T_thr: dict[str, float], T_lat: dict[str, float],
               M: int = 1) -> dict[str, float]:
    N = n // nb
    b = {"area": area(N, T_thr, M), "chain": chain(N, T_lat),
         "critical_path": critical_path(N, T_lat) if N <= 64 else float("nan"),
         "gemm_peak": gemm_peak(n, nb, T_thr["GEMM"], M)}
    b["mixed"] = max(b["area"], b["chain"])
    return b


def lp_area_mixed(N: int, T: dict[str, dict[str, float]], M: dict[str, int],
                  mixed_chain: bool = True) -> float:
    """General LP of L349-359 (+ chain constraint L388-396 if mixed_chain) over
    resource types r with times T[r][t] and counts M[r]; returns l*.
    Variables x = [n_rt for r, t] + [l]."""
    from scipy.optimize import linprog
    types = ["POTRF", "TRSM", "SYRK", "GEMM"]
    res = list(T.keys())
    c_ = task_counts(N)
    nv = len(res) * len(types) + 1
    idx = lambda r, t: res.index(r) * len(types) + types.index(t)
    cost = [0.0] * nv
    cost[-1] = 1.0
    A_eq, b_eq, A_ub, b_ub = [], [], [], []
    for t in types:  # sum_r n_rt = N_t
        row = [0.0] * nv
        for r in res:
            row[idx(r, t)] = 1.0
        A_eq.append(row)
        b_eq.append(c_[t])
    for r in res:  # sum_t n_rt T_rt <= l M_r
        row = [0.0] * nv
        for t in types:
            row[idx(r, t)] = T[r][t]
        row[-1] = -float(M[r])
        A_ub.append(row)
        b_ub.append(0.0)
    if mixed_chain:
        row = [0.0] * nv
        for r in res:
            row[idx(r, "POTRF")] = T[r]["POTRF"]
        row[-1] = -1.0
        tT = min(T[r]["TRSM"] for r in res)
        tS = min(T[r]["SYRK"] for r in res)
        A_ub.append(row)
        b_ub.append(-(N - 1) * (tT + tS))
    sol = linprog(cost, A_ub=A_ub, b_ub=b_ub, A_eq=A_eq, b_eq=b_eq,
                  bounds=[(0, None)] * nv, method="highs")
    assert sol.status == 0, sol.message
    return float(sol.x[-1])


def owner_area(N: int, p: int, q: int, T_thr: dict[str, float]) -> tuple[float, list[float]]:
    """Owner-area bound (ext): every task of the brute-force task list runs on
    the owner (i mod p, j mod q) of the tile it writes (owner-computes, L263-274); the
    busiest rank's summed T_thr bounds any schedule on that grid."""
    w = [0.0] * (p * q)
    for t in dag.tasks(N):
        i, j = t.writes
        w[(i % p) * q + (j % q)] += T_thr[dag.TYPE_NAMES[t.type]]
    return max(w), w
