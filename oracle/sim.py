"""ORACLE -- TEST INFRASTRUCTURE ONLY.  Plain-Python replay of the Algorithm 1 task DAG on a
platform of resource classes, written from the paper's scheduler descriptions:

* dmda: "each task is assigned to the processing resource which is
  estimated to complete it first" -- the estimate is the time the worker's already
  assigned tasks end plus the task's execution time on the worker's class; tasks are
  assigned when they become ready (StarPU pushes them to per-worker queues), in release
  order, and a worker runs its queue in order.
* dmdas (L652-660): the same, but ready tasks are assigned, and each worker's queue is
  served, in priority order; the priority is the longest path to an exit task with each
  task's fastest execution time over the resources.
* static rules: GEMM/SYRK forced on one class (L1000-1007); TRSMs at least d tiles below
  the diagonal forced on another (L1019-1025).

No data transfers are modelled (reading R18).  Tie-breaking (a convention the
paper leaves open, shared with the library so results compare exactly): completions at
the same instant are all processed before any assignment; ties in completion estimate go
to the lowest worker number (workers numbered class by class); equal priorities keep
release order (task id).  Only tests/ may import this module.
"""
from __future__ import annotations

import math

from . import dag


def _runs_on(cls: int, task: dag.Task, times, gemm_syrk_class: int, trsm_far_class: int, trsm_far_distance: int):
    t = times[cls][task.type]
    if not (t >= 0) or math.isinf(t):
        return False
    if gemm_syrk_class >= 0 and task.type in (dag.SYRK, dag.GEMM) and cls != gemm_syrk_class:
        return False
    if trsm_far_class >= 0 and task.type == dag.TRSM and task.i - task.k >= trsm_far_distance and cls != trsm_far_class:
        return False
    return True


def simulate(N: int, workers, times, policy: int = 1, gemm_syrk_class: int = -1, trsm_far_class: int = -1,
             trsm_far_distance: int = 1):
    """Returns (makespan, {task index: (worker, class, t0, t1)}); policy 0 = dmda, 1 = dmdas."""
    ts, E = dag.edges(N)
    wcls = [r for r, m in enumerate(workers) for _ in range(m)]
    W = len(wcls)
    succ = [[] for _ in ts]
    indeg = [0] * len(ts)
    for a, b in E:
        succ[a].append(b)
        indeg[b] += 1
    fastest = []
    for t in range(4):
        v = [times[r][t] for r in range(len(workers)) if workers[r] > 0 and times[r][t] >= 0 and not math.isinf(times[r][t])]
        fastest.append(min(v) if v else 0.0)
    prio = dag.bottom_levels(N, lambda task: fastest[task.type])
    queue = [[] for _ in range(W)]
    exp_free = [0.0] * W
    running = [None] * W  # (end, task)
    out = {}

    def assign(ready, now):
        if policy == 1:
            ready = sorted(ready, key=lambda x: -prio[x])  # stable: release order among equals
        for x in ready:
            best, bend = None, None
            for w in range(W):
                if not _runs_on(wcls[w], ts[x], times, gemm_syrk_class, trsm_far_class, trsm_far_distance):
                    continue
                end = max(exp_free[w], now) + times[wcls[w]][ts[x].type]
                if best is None or end < bend:
                    best, bend = w, end
            assert best is not None, "a task no class may run"
            queue[best].append(x)
            exp_free[best] = bend

    def start(now):
        for w in range(W):
            if running[w] is not None or not queue[w]:
                continue
            pick = 0
            if policy == 1:
                for q in range(1, len(queue[w])):
                    if prio[queue[w][q]] > prio[queue[w][pick]]:
                        pick = q
            x = queue[w].pop(pick)
            end = now + times[wcls[w]][ts[x].type]
            running[w] = (end, x)
            out[x] = (w, wcls[w], now, end)

    assign([x for x in range(len(ts)) if indeg[x] == 0], 0.0)
    start(0.0)
    makespan = 0.0
    while any(r is not None for r in running):
        now = min(r[0] for r in running if r is not None)
        ready = []
        for w in range(W):  # all completions at this instant, in worker order
            if running[w] is not None and running[w][0] == now:
                x = running[w][1]
                running[w] = None
                makespan = max(makespan, now)
                for s in succ[x]:
                    indeg[s] -= 1
                    if indeg[s] == 0:
                        ready.append(s)
        assign(ready, now)
        start(now)
    assert len(out) == len(ts)
    return makespan, out
