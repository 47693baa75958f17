"""ORACLE -- TEST INFRASTRUCTURE ONLY.  Brute-force minimum makespan of the Algorithm 1 task
DAG on a small platform of resource classes (the paper's constraint-
programming formulation: one resource per task, start times, resource
capacity, dependencies, no transfers).

Exhaustive: every topological order of the tasks times every assignment of tasks to workers
(allowed classes only), each placed greedily (start = max(predecessors' finish, the
worker's previous task's finish)) -- this enumerates every semi-active schedule, and some
semi-active schedule is optimal (left-shifting a schedule never increases its makespan).
Tiny instances only (N <= 3, a handful of workers).  Only tests/ may import this module.
"""
from __future__ import annotations

import itertools
import math

from . import dag


def _allowed(task: dag.Task, cls: int, times, gemm_syrk_class: int, trsm_far_class: int, trsm_far_distance: int):
    t = times[cls][task.type]
    if not (t >= 0) or math.isinf(t):
        return False
    if gemm_syrk_class >= 0 and task.type in (dag.SYRK, dag.GEMM) and cls != gemm_syrk_class:
        return False
    if trsm_far_class >= 0 and task.type == dag.TRSM and task.i - task.k >= trsm_far_distance and cls != trsm_far_class:
        return False
    return True


def topological_orders(n: int, preds):
    """Every topological order of tasks 0..n-1 (preds[t] = predecessors)."""
    indeg = [len(p) for p in preds]
    succ = [[] for _ in range(n)]
    for t in range(n):
        for p in preds[t]:
            succ[p].append(t)
    order = []

    def rec():
        if len(order) == n:
            yield list(order)
            return
        for t in range(n):
            if indeg[t] == 0 and t not in order:
                order.append(t)
                for s in succ[t]:
                    indeg[s] -= 1
                yield from rec()
                for s in succ[t]:
                    indeg[s] += 1
                order.pop()

    yield from rec()


def optimal_makespan(N: int, workers, times, gemm_syrk_class: int = -1, trsm_far_class: int = -1,
                     trsm_far_distance: int = 1) -> float:
    ts, E = dag.edges(N)
    n = len(ts)
    preds = [[] for _ in range(n)]
    for a, b in E:
        preds[b].append(a)
    wcls = [r for r, m in enumerate(workers) for _ in range(m)]
    options = [[w for w in range(len(wcls)) if _allowed(ts[t], wcls[w], times, gemm_syrk_class, trsm_far_class,
                                                         trsm_far_distance)] for t in range(n)]
    orders = list(topological_orders(n, preds))
    best = math.inf
    for assign in itertools.product(*options):
        for order in orders:
            free = [0.0] * len(wcls)
            fin = [0.0] * n
            for t in order:
                w = assign[t]
                start = max([free[w]] + [fin[p] for p in preds[t]])
                fin[t] = start + times[wcls[w]][ts[t].type]
                free[w] = fin[t]
            best = min(best, max(fin))
    return best
