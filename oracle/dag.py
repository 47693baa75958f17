"""ORACLE -- TEST INFRASTRUCTURE ONLY.  The task graph of the tiled Cholesky.

* Tasks: Algorithm 1 enumerated in program order, named as
  in Fig. 1 (L221-257): ``POTRF_k``, ``TRSM_i_k``, ``SYRK_j_k``, ``GEMM_i_j_k``.
* Edges: "direct data dependency" (L213-220).  Derived here by brute force from
  each task's read / write tile sets in program order (the way StarPU infers
  them from access modes, L523-552): a task depends on the last writer of every
  tile it reads or writes.  Nothing about the Cholesky structure is assumed.
* Weights / priorities: bottom-level = weight of the longest path from a task to
  an exit task, the task's own weight included (HEFT, L299-301; dmdas, L655-660;
  reading R13).

This module shares no code with the CUDA library.
"""
from __future__ import annotations

from dataclasses import dataclass

POTRF, TRSM, SYRK, GEMM = 0, 1, 2, 3
TYPE_NAMES = ("POTRF", "TRSM", "SYRK", "GEMM")


@dataclass(frozen=True)
class Task:
    type: int
    i: int
    j: int
    k: int

    @property
    def name(self) -> str:  # Fig. 1 naming
        if self.type == POTRF:
            return f"POTRF_{self.k}"
        if self.type == TRSM:
            return f"TRSM_{self.i}_{self.k}"
        if self.type == SYRK:
            return f"SYRK_{self.j}_{self.k}"
        return f"GEMM_{self.i}_{self.j}_{self.k}"

    @property
    def writes(self) -> tuple[int, int]:
        return {POTRF: (self.k, self.k), TRSM: (self.i, self.k),
                SYRK: (self.j, self.j), GEMM: (self.i, self.j)}[self.type]

    @property
    def reads(self) -> tuple[tuple[int, int], ...]:
        if self.type == POTRF:
            return ((self.k, self.k),)
        if self.type == TRSM:
            return ((self.k, self.k), (self.i, self.k))
        if self.type == SYRK:
            return ((self.j, self.k), (self.j, self.j))
        return ((self.i, self.k), (self.j, self.k), (self.i, self.j))


def tasks(N: int) -> list[Task]:
    """Algorithm 1, program order (reading R2: GEMM loop nested in the j loop)."""
    out: list[Task] = []
    for k in range(N):
        out.append(Task(POTRF, k, k, k))
        for i in range(k + 1, N):
            out.append(Task(TRSM, i, k, k))
        for j in range(k + 1, N):
            out.append(Task(SYRK, j, j, k))
            for i in range(j + 1, N):
                out.append(Task(GEMM, i, j, k))
    return out


def edges(N: int) -> tuple[list[Task], list[tuple[int, int]]]:
    """Brute-force direct dependencies from read/write sets; returns (tasks, edge list
    as (pred index, succ index) into the task list)."""
    ts = tasks(N)
    last_writer: dict[tuple[int, int], int] = {}
    E: list[tuple[int, int]] = []
    for idx, t in enumerate(ts):
        preds = set()
        for tile in set(t.reads) | {t.writes}:
            w = last_writer.get(tile)
            if w is not None:
                preds.add(w)
        for p in sorted(preds):
            E.append((p, idx))
        last_writer[t.writes] = idx
    return ts, E


def counts(N: int) -> dict[str, int]:
    c = {n: 0 for n in TYPE_NAMES}
    for t in tasks(N):
        c[TYPE_NAMES[t.type]] += 1
    return c


def in_degrees(N: int) -> list[int]:
    ts, E = edges(N)
    deg = [0] * len(ts)
    for _, s in E:
        deg[s] += 1
    return deg


def longest_path(N: int, weight) -> float:
    """Weight of the longest path through the DAG (a task's weight = weight(task))."""
    ts, E = edges(N)
    succ: list[list[int]] = [[] for _ in ts]
    for p, s in E:
        succ[p].append(s)
    best = [0.0] * len(ts)
    for idx in range(len(ts) - 1, -1, -1):  # program order is topological
        tail = max((best[s] for s in succ[idx]), default=0.0)
        best[idx] = weight(ts[idx]) + tail
    return max(best) if best else 0.0


def bottom_levels(N: int, weight) -> list[float]:
    """Bottom-level of every task (own weight included), program order."""
    ts, E = edges(N)
    succ: list[list[int]] = [[] for _ in ts]
    for p, s in E:
        succ[p].append(s)
    bl = [0.0] * len(ts)
    for idx in range(len(ts) - 1, -1, -1):
        bl[idx] = weight(ts[idx]) + max((bl[s] for s in succ[idx]), default=0.0)
    return bl


def acceleration_factor_K(N: int, a=(2.0, 11.0, 26.0, 29.0)) -> float:
    """K = (N_P a_P + N_T a_T + N_S a_S + N_G a_G) / total tasks,
    with Table I's factors POTRF 2x, TRSM 11x, SYRK 26x, GEMM 29x (L784-787)."""
    c = counts(N)
    tot = sum(c.values())
    return (c["POTRF"] * a[0] + c["TRSM"] * a[1] + c["SYRK"] * a[2] + c["GEMM"] * a[3]) / tot
