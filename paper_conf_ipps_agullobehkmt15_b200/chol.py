"""Thin ctypes binding of libchol_b200.so (include/chol.h) -- argument marshalling only.

Every function has the C name and returns what the C call returns (status codes are
turned into ``CholError`` exceptions).  Matrices are passed as raw pointers taken from
torch tensors (``data_ptr()``, device or pinned host memory) or numpy arrays (host).
There is no CPU fallback: if the CUDA library is missing this module raises on import.
"""
from __future__ import annotations

import ctypes
import os

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("CHOL_LIB_OVERRIDE") or os.path.join(_HERE, "libchol_b200.so")  # override: A/B experiments only

POLICY_CP_PRIORITY, POLICY_DYNAMIC, POLICY_STATIC = 0, 1, 2  # zero-initialised opts = CP_PRIORITY
EXEC_SCHEDULER, EXEC_HOST = 0, 1
POTRF, TRSM, SYRK, GEMM = 0, 1, 2, 3
TYPE_NAMES = ("POTRF", "TRSM", "SYRK", "GEMM")


class CholError(RuntimeError):
    def __init__(self, status: int, what: str):
        self.status = status
        super().__init__(f"{what}: status {status} ({chol_strerror(status)})")


class chol_opts_t(ctypes.Structure):
    _fields_ = [("policy", ctypes.c_int), ("trsm_pin_distance", ctypes.c_int),
                ("latency_workers", ctypes.c_int), ("grid_p", ctypes.c_int), ("grid_q", ctypes.c_int),
                ("trace", ctypes.c_int), ("executor", ctypes.c_int), ("workers", ctypes.c_int),
                ("cpu_trsm_distance", ctypes.c_int), ("cpu_threads", ctypes.c_int)]


class chol_task_rec_t(ctypes.Structure):
    _fields_ = [("type", ctypes.c_uint8), ("gpu", ctypes.c_uint8), ("worker", ctypes.c_uint16),
                ("i", ctypes.c_int32), ("j", ctypes.c_int32), ("k", ctypes.c_int32),
                ("t0_ns", ctypes.c_uint64), ("t1_ns", ctypes.c_uint64)]


SIM_MAX_CLASSES = 4
SIM_DMDA, SIM_DMDAS, SIM_FIXED = 0, 1, 2


class chol_sim_opts_t(ctypes.Structure):
    _fields_ = [("nclasses", ctypes.c_int), ("workers", ctypes.c_int * SIM_MAX_CLASSES),
                ("time", (ctypes.c_double * 4) * SIM_MAX_CLASSES), ("policy", ctypes.c_int),
                ("gemm_syrk_class", ctypes.c_int), ("trsm_far_class", ctypes.c_int),
                ("trsm_far_distance", ctypes.c_int), ("fixed_worker", ctypes.POINTER(ctypes.c_int32)),
                ("fixed_rank", ctypes.POINTER(ctypes.c_int32))]


def _load():
    if not os.path.exists(LIB_PATH):
        raise ImportError(f"{LIB_PATH} is missing: run __graft_entry__.build() (there is no CPU fallback)")
    L = ctypes.CDLL(LIB_PATH)
    P, i64, i32, u64, vp = ctypes.c_void_p, ctypes.c_int64, ctypes.c_int, ctypes.c_uint64, ctypes.c_void_p
    dp = ctypes.POINTER(ctypes.c_double)
    sig = {
        "chol_plan": ([i64, i64, i32, ctypes.POINTER(P)], i32),
        "chol_plan_ex": ([i64, i64, i32, ctypes.POINTER(chol_opts_t), ctypes.POINTER(P)], i32),
        "chol_factor": ([P, vp, i64, vp, i64, ctypes.POINTER(i32)], i32),
        "chol_trace": ([P, ctypes.POINTER(chol_task_rec_t), i64, ctypes.POINTER(i64), dp], i32),
        "chol_destroy": ([P], i32),
        "chol_strerror": ([i32], ctypes.c_char_p),
        "chol_generate": ([P, u64, i32], i32),
        "chol_scatter": ([P, vp, i64], i32),
        "chol_gather": ([P, vp, i64], i32),
        "chol_owner_area": ([i64, i32, i32, dp, dp, dp], i32),
        "chol_scatter_tiles": ([P, vp, i64], i32),
        "chol_gather_tiles": ([P, vp, i64], i32),
        "chol_factor_inplace": ([P, ctypes.POINTER(i32)], i32),
        "chol_last_times": ([P, dp, dp], i32),
        "chol_get_stream": ([P, ctypes.POINTER(vp)], i32),
        "chol_get_info": ([P, ctypes.POINTER(i64), ctypes.POINTER(i64), ctypes.POINTER(i32),
                           ctypes.POINTER(i32), ctypes.POINTER(i32), ctypes.POINTER(i32)], i32),
        "chol_run_task": ([P, i32, i32, i32, i32, i32, dp], i32),
        "chol_run_batch": ([P, i32, i32, i32, dp], i32),
        "chol_last_launches": ([P, ctypes.POINTER(i32)], i32),
        "chol_dag": ([i64, ctypes.POINTER(i64), ctypes.POINTER(i64), ctypes.POINTER(i64), i64], i32),
        "chol_task_id": ([i64, i32, i32, i32, i32, ctypes.POINTER(i64)], i32),
        "chol_bounds": ([i64, i64, i32, dp, dp, dp], i32),
        "chol_job_trace": ([P, ctypes.POINTER(ctypes.c_uint64), i64, ctypes.POINTER(i64)], i32),
        "chol_job_desc": ([P, ctypes.POINTER(ctypes.c_int32), i64, ctypes.POINTER(i64)], i32),
        "chol_plan_dist": ([i64, i64, i32, i32, ctypes.POINTER(chol_opts_t), ctypes.POINTER(P)], i32),
        "chol_dist_export": ([P, vp, i64, ctypes.POINTER(i64)], i32),
        "chol_dist_connect": ([P, vp, i64], i32),
        "chol_get_dist": ([P, ctypes.POINTER(i32), ctypes.POINTER(i32), ctypes.POINTER(i32), ctypes.POINTER(i32),
                           ctypes.POINTER(i64), ctypes.POINTER(i64)], i32),
        "chol_factor_async": ([P], i32),
        "chol_wait": ([P, ctypes.POINTER(i32)], i32),
        "chol_dist_layout": ([i64, i64, i32, i32, i32, ctypes.POINTER(i32), ctypes.POINTER(i32),
                              ctypes.POINTER(ctypes.c_int32), i64], i32),
        "chol_lp_bound": ([i64, i32, ctypes.POINTER(i32), dp, i32, dp, dp], i32),
        "chol_solve": ([P, vp, i64, i64], i32),
        "chol_last_solve_times": ([P, dp, dp], i32),
        "chol_simulate": ([i64, ctypes.POINTER(chol_sim_opts_t), dp, ctypes.POINTER(chol_task_rec_t), i64], i32),
        "chol_set_task_priorities": ([P, dp, i64], i32),
        "chol_cpu_trsm": ([vp, vp, i64, i32], i32),
        "chol_optimal_schedule": ([i64, ctypes.POINTER(chol_sim_opts_t), i64, dp, ctypes.POINTER(i32),
                                   ctypes.POINTER(ctypes.c_int32), ctypes.POINTER(ctypes.c_int32),
                                   ctypes.POINTER(i64)], i32),
    }
    for name, (args, res) in sig.items():
        f = getattr(L, name)
        f.argtypes = args
        f.restype = res
    return L


_lib = _load()
EXPORTED = ("chol_plan", "chol_plan_ex", "chol_factor", "chol_trace", "chol_destroy", "chol_strerror",
            "chol_generate", "chol_scatter", "chol_gather", "chol_factor_inplace", "chol_last_times",
            "chol_get_stream", "chol_get_info", "chol_run_task", "chol_run_batch", "chol_last_launches",
            "chol_dag", "chol_task_id", "chol_bounds", "chol_job_trace", "chol_job_desc", "chol_plan_dist", "chol_dist_export",
            "chol_dist_connect", "chol_get_dist", "chol_factor_async", "chol_wait", "chol_dist_layout",
            "chol_lp_bound", "chol_simulate", "chol_solve", "chol_last_solve_times", "chol_scatter_tiles",
            "chol_gather_tiles", "chol_owner_area", "chol_optimal_schedule", "chol_set_task_priorities",
            "chol_cpu_trsm")


def _ptr(x) -> int:
    """Raw address of a torch tensor / numpy array / int."""
    if isinstance(x, int):
        return x
    if hasattr(x, "data_ptr"):
        return x.data_ptr()
    if hasattr(x, "ctypes"):
        return x.ctypes.data
    raise TypeError(f"cannot take a pointer of {type(x)}")


def _check(st: int, what: str) -> None:
    if st != 0:
        raise CholError(st, what)


def chol_strerror(status: int) -> str:
    return _lib.chol_strerror(status).decode()


def chol_plan(n: int, nb: int, ngpus: int = 1) -> int:
    h = ctypes.c_void_p()
    _check(_lib.chol_plan(n, nb, ngpus, ctypes.byref(h)), "chol_plan")
    return h.value


def chol_plan_ex(n: int, nb: int, ngpus: int = 1, **opts) -> int:
    o = chol_opts_t(**opts)
    h = ctypes.c_void_p()
    _check(_lib.chol_plan_ex(n, nb, ngpus, ctypes.byref(o), ctypes.byref(h)), "chol_plan_ex")
    return h.value


def chol_factor(plan: int, A, lda: int, L, ldl: int) -> int:
    info = ctypes.c_int(0)
    _check(_lib.chol_factor(plan, _ptr(A), lda, _ptr(L), ldl, ctypes.byref(info)), "chol_factor")
    return info.value


def chol_factor_inplace(plan: int) -> int:
    info = ctypes.c_int(0)
    _check(_lib.chol_factor_inplace(plan, ctypes.byref(info)), "chol_factor_inplace")
    return info.value


def chol_trace(plan: int):
    """Returns (records as a list of dicts, makespan in seconds)."""
    n = ctypes.c_int64(0)
    ms = ctypes.c_double(0.0)
    _check(_lib.chol_trace(plan, None, 0, ctypes.byref(n), ctypes.byref(ms)), "chol_trace")
    recs = (chol_task_rec_t * max(n.value, 1))()
    _check(_lib.chol_trace(plan, recs, n.value, ctypes.byref(n), ctypes.byref(ms)), "chol_trace")
    out = [{"type": r.type, "gpu": r.gpu, "worker": r.worker, "i": r.i, "j": r.j, "k": r.k,
            "t0_ns": r.t0_ns, "t1_ns": r.t1_ns} for r in recs[:n.value]]
    return out, ms.value


def chol_job_trace(plan: int):
    """numpy array (njobs, 5): t0_ns, t1_ns, worker << 32 | smid, type << 32 | task id, t_enqueue_ns."""
    import numpy as np
    n = ctypes.c_int64(0)
    _check(_lib.chol_job_trace(plan, None, 0, ctypes.byref(n)), "chol_job_trace")
    out = np.zeros((max(n.value, 1), 5), dtype=np.uint64)
    _check(_lib.chol_job_trace(plan, out.ctypes.data_as(ctypes.POINTER(ctypes.c_uint64)), n.value,
                               ctypes.byref(n)), "chol_job_trace")
    return out[:n.value]


def chol_job_desc(plan: int):
    """numpy array (njobs, 8) int32: type, i, j, k, a, b, c, node (include/chol.h)."""
    import numpy as np
    n = ctypes.c_int64(0)
    _check(_lib.chol_job_desc(plan, None, 0, ctypes.byref(n)), "chol_job_desc")
    out = np.zeros((max(n.value, 1), 8), dtype=np.int32)
    _check(_lib.chol_job_desc(plan, out.ctypes.data_as(ctypes.POINTER(ctypes.c_int32)), n.value,
                              ctypes.byref(n)), "chol_job_desc")
    return out[:n.value]


def chol_destroy(plan: int) -> None:
    _check(_lib.chol_destroy(plan), "chol_destroy")


def chol_generate(plan: int, seed: int, family: int = 0) -> None:
    _check(_lib.chol_generate(plan, seed, family), "chol_generate")


def chol_scatter(plan: int, A, lda: int) -> None:
    _check(_lib.chol_scatter(plan, _ptr(A), lda), "chol_scatter")


def chol_gather(plan: int, L, ldl: int) -> None:
    _check(_lib.chol_gather(plan, _ptr(L), ldl), "chol_gather")


def chol_scatter_tiles(plan: int, tiles, count: int) -> None:
    """The plan's OWNED tiles, packed nb x nb in Algorithm 1 tile order (host or device)."""
    _check(_lib.chol_scatter_tiles(plan, _ptr(tiles), count), "chol_scatter_tiles")


def chol_gather_tiles(plan: int, tiles, count: int) -> None:
    _check(_lib.chol_gather_tiles(plan, _ptr(tiles), count), "chol_gather_tiles")


def chol_last_times(plan: int) -> tuple[float, float]:
    f, l = ctypes.c_double(), ctypes.c_double()
    _check(_lib.chol_last_times(plan, ctypes.byref(f), ctypes.byref(l)), "chol_last_times")
    return f.value, l.value


def chol_get_stream(plan: int) -> int:
    s = ctypes.c_void_p()
    _check(_lib.chol_get_stream(plan, ctypes.byref(s)), "chol_get_stream")
    return s.value or 0


def chol_get_info(plan: int) -> dict:
    n, nb = ctypes.c_int64(), ctypes.c_int64()
    bs, w, pol, ex = ctypes.c_int(), ctypes.c_int(), ctypes.c_int(), ctypes.c_int()
    _check(_lib.chol_get_info(plan, ctypes.byref(n), ctypes.byref(nb), ctypes.byref(bs), ctypes.byref(w),
                              ctypes.byref(pol), ctypes.byref(ex)), "chol_get_info")
    return {"n": n.value, "nb": nb.value, "block": bs.value, "workers": w.value, "policy": pol.value,
            "executor": ex.value}


def chol_run_task(plan: int, type: int, i: int, j: int, k: int, reps: int = 1) -> float:
    ms = ctypes.c_double()
    _check(_lib.chol_run_task(plan, type, i, j, k, reps, ctypes.byref(ms)), "chol_run_task")
    return ms.value


def chol_run_batch(plan: int, type: int, count: int, reps: int = 1) -> float:
    ms = ctypes.c_double()
    _check(_lib.chol_run_batch(plan, type, count, reps, ctypes.byref(ms)), "chol_run_batch")
    return ms.value


def chol_set_task_priorities(plan: int, prio) -> None:
    """Static priorities per task (chol_task_id order, higher first) for the device scheduler."""
    arr = (ctypes.c_double * len(prio))(*[float(v) for v in prio])
    _check(_lib.chol_set_task_priorities(plan, arr, len(prio)), "chol_set_task_priorities")


def chol_cpu_trsm(X, L, bs: int = 96) -> None:
    """X <- X L^{-T} on the host CPU (the NEXT-3 class's tile kernel); X, L numpy (nb x nb)."""
    nb = X.shape[0]
    _check(_lib.chol_cpu_trsm(_ptr(X), _ptr(L), nb, bs), "chol_cpu_trsm")


def chol_last_launches(plan: int) -> int:
    n = ctypes.c_int()
    _check(_lib.chol_last_launches(plan, ctypes.byref(n)), "chol_last_launches")
    return n.value


def chol_dag(N: int):
    """(ntasks, edges as a list of (pred, succ) dense task ids)."""
    nt, ne = ctypes.c_int64(), ctypes.c_int64()
    _check(_lib.chol_dag(N, ctypes.byref(nt), ctypes.byref(ne), None, 0), "chol_dag")
    buf = (ctypes.c_int64 * max(2 * ne.value, 1))()
    _check(_lib.chol_dag(N, ctypes.byref(nt), ctypes.byref(ne), buf, ne.value), "chol_dag")
    return nt.value, [(buf[2 * e], buf[2 * e + 1]) for e in range(ne.value)]


def chol_task_id(N: int, type: int, i: int, j: int, k: int) -> int:
    v = ctypes.c_int64()
    _check(_lib.chol_task_id(N, type, i, j, k, ctypes.byref(v)), "chol_task_id")
    return v.value


BOUND_NAMES = ("area", "chain", "mixed", "critical_path", "gemm_peak", "max_area_cp")


def chol_bounds(n: int, nb: int, ngpus: int, T_lat, T_thr) -> dict:
    """Makespan lower bounds (seconds) from per-type times [POTRF, TRSM, SYRK, GEMM]."""
    lat = (ctypes.c_double * 4)(*T_lat)
    thr = (ctypes.c_double * 4)(*T_thr)
    out = (ctypes.c_double * 6)()
    _check(_lib.chol_bounds(n, nb, ngpus, lat, thr, out), "chol_bounds")
    return dict(zip(BOUND_NAMES, list(out)))


def chol_solve(plan: int, B, ldb: int, nrhs: int) -> None:
    """A X = B with the plan's factor; B (n x nrhs row-major, host or device) is overwritten."""
    _check(_lib.chol_solve(plan, _ptr(B), ldb, nrhs), "chol_solve")


def chol_last_solve_times(plan: int) -> tuple[float, float]:
    a, b = ctypes.c_double(), ctypes.c_double()
    _check(_lib.chol_last_solve_times(plan, ctypes.byref(a), ctypes.byref(b)), "chol_last_solve_times")
    return a.value, b.value


def chol_owner_area(N: int, p: int, q: int, T_thr) -> tuple[float, list]:
    """Owner-area bound on a p x q block-cyclic grid: (max over ranks, per-rank sums)."""
    tt = (ctypes.c_double * 4)(*[T_thr[k] for k in ("POTRF", "TRSM", "SYRK", "GEMM")]) \
        if isinstance(T_thr, dict) else (ctypes.c_double * 4)(*T_thr)
    out = ctypes.c_double()
    per = (ctypes.c_double * (p * q))()
    _check(_lib.chol_owner_area(N, p, q, tt, ctypes.byref(out), per), "chol_owner_area")
    return out.value, list(per)


def chol_lp_bound(N: int, workers, times, mixed: bool = True):
    """LP makespan bound over resource classes: workers[r], times[r] =
    [POTRF, TRSM, SYRK, GEMM] seconds (negative / inf = cannot run).  Returns (l, n_rt)."""
    R = len(workers)
    w = (ctypes.c_int * R)(*workers)
    t = (ctypes.c_double * (4 * R))(*[float(v) for row in times for v in row])
    l = ctypes.c_double()
    nrt = (ctypes.c_double * (4 * R))()
    _check(_lib.chol_lp_bound(N, R, w, t, int(bool(mixed)), ctypes.byref(l), nrt), "chol_lp_bound")
    return l.value, [list(nrt[4 * r:4 * r + 4]) for r in range(R)]


def _sim_opts(workers, times, policy, gemm_syrk_class, trsm_far_class, trsm_far_distance, fixed=None):
    o = chol_sim_opts_t()
    o.nclasses = len(workers)
    for r, (m, row) in enumerate(zip(workers, times)):
        o.workers[r] = m
        for t in range(4):
            o.time[r][t] = float(row[t])
    o.policy, o.gemm_syrk_class, o.trsm_far_class, o.trsm_far_distance = policy, gemm_syrk_class, trsm_far_class, \
        trsm_far_distance
    keep = None
    if fixed is not None:
        w, r = fixed
        keep = ((ctypes.c_int32 * len(w))(*w), (ctypes.c_int32 * len(r))(*r))
        o.fixed_worker = ctypes.cast(keep[0], ctypes.POINTER(ctypes.c_int32))
        o.fixed_rank = ctypes.cast(keep[1], ctypes.POINTER(ctypes.c_int32))
    return o, keep


def chol_simulate(N: int, workers, times, policy: int = SIM_DMDAS, gemm_syrk_class: int = -1,
                  trsm_far_class: int = -1, trsm_far_distance: int = 1, records: bool = False, fixed=None):
    """Replay of the Algorithm 1 DAG on a platform of resource classes under dmda / dmdas,
    the paper's static rules, or an injected schedule (policy SIM_FIXED, fixed = (worker per
    task, rank per task)) -- chol_simulate in include/chol.h.  Returns the makespan (seconds)
    and, with records=True, the per-task records (chol_task_id order)."""
    o, keep = _sim_opts(workers, times, policy, gemm_syrk_class, trsm_far_class, trsm_far_distance, fixed)
    mk = ctypes.c_double()
    nt = N + N * (N - 1) + N * (N - 1) * (N - 2) // 6
    recs = (chol_task_rec_t * nt)() if records else None
    _check(_lib.chol_simulate(N, ctypes.byref(o), ctypes.byref(mk), recs, nt if records else 0), "chol_simulate")
    if not records:
        return mk.value
    return mk.value, [{"type": r.type, "cls": r.gpu, "worker": r.worker, "i": r.i, "j": r.j, "k": r.k,
                       "t0_ns": r.t0_ns, "t1_ns": r.t1_ns} for r in recs]


def chol_optimal_schedule(N: int, workers, times, gemm_syrk_class: int = -1, trsm_far_class: int = -1,
                          trsm_far_distance: int = 1, node_limit: int = 0):
    """Exact minimum-makespan schedule (branch and bound, include/chol.h).  Returns
    (makespan, optimal, worker per task, rank per task, search nodes)."""
    o, _ = _sim_opts(workers, times, SIM_DMDAS, gemm_syrk_class, trsm_far_class, trsm_far_distance)
    nt = N + N * (N - 1) + N * (N - 1) * (N - 2) // 6
    mk, opt, nodes = ctypes.c_double(), ctypes.c_int(), ctypes.c_int64()
    w, r = (ctypes.c_int32 * nt)(), (ctypes.c_int32 * nt)()
    _check(_lib.chol_optimal_schedule(N, ctypes.byref(o), node_limit, ctypes.byref(mk), ctypes.byref(opt), w, r,
                                      ctypes.byref(nodes)), "chol_optimal_schedule")
    return mk.value, bool(opt.value), list(w), list(r), nodes.value


def chol_plan_dist(n: int, nb: int, nranks: int, rank: int, **opts) -> int:
    o = chol_opts_t(**opts)
    h = ctypes.c_void_p()
    _check(_lib.chol_plan_dist(n, nb, nranks, rank, ctypes.byref(o), ctypes.byref(h)), "chol_plan_dist")
    return h.value


def chol_dist_export(plan: int) -> bytes:
    ln = ctypes.c_int64()
    _check(_lib.chol_dist_export(plan, None, 0, ctypes.byref(ln)), "chol_dist_export")
    buf = ctypes.create_string_buffer(ln.value)
    _check(_lib.chol_dist_export(plan, buf, ln.value, ctypes.byref(ln)), "chol_dist_export")
    return buf.raw


def chol_dist_connect(plan: int, blobs: list) -> None:
    stride = len(blobs[0])
    assert all(len(b) == stride for b in blobs)
    joined = ctypes.create_string_buffer(b"".join(blobs), stride * len(blobs))
    _check(_lib.chol_dist_connect(plan, joined, stride), "chol_dist_connect")


def chol_get_dist(plan: int) -> dict:
    r, nr, gp, gq = ctypes.c_int(), ctypes.c_int(), ctypes.c_int(), ctypes.c_int()
    no, ns = ctypes.c_int64(), ctypes.c_int64()
    _check(_lib.chol_get_dist(plan, ctypes.byref(r), ctypes.byref(nr), ctypes.byref(gp), ctypes.byref(gq),
                              ctypes.byref(no), ctypes.byref(ns)), "chol_get_dist")
    return {"rank": r.value, "nranks": nr.value, "grid_p": gp.value, "grid_q": gq.value, "nowned": no.value,
            "nslots": ns.value}


def chol_factor_async(plan: int) -> None:
    _check(_lib.chol_factor_async(plan), "chol_factor_async")


def chol_wait(plan: int) -> int:
    info = ctypes.c_int(0)
    _check(_lib.chol_wait(plan, ctypes.byref(info)), "chol_wait")
    return info.value


def chol_dist_layout(n: int, nb: int, p: int, q: int, rank: int):
    """(nowned, ncached, slot_map list) of a rank of the p x q grid (host only)."""
    no, nc = ctypes.c_int(), ctypes.c_int()
    N = n // nb
    sm = (ctypes.c_int32 * max(N * (N + 1) // 2, 1))()
    _check(_lib.chol_dist_layout(n, nb, p, q, rank, ctypes.byref(no), ctypes.byref(nc), sm, N * (N + 1) // 2),
           "chol_dist_layout")
    return no.value, nc.value, list(sm[:N * (N + 1) // 2])


class DistPlan:
    """One rank of a multi-GPU factorization.  `allgather(bytes) -> list[bytes]` exchanges
    the connection blobs (e.g. torch.distributed.all_gather_object); for logical ranks in
    one process build all plans first and connect them with connect_local()."""

    def __init__(self, n: int, nb: int, nranks: int, rank: int, allgather=None, **opts):
        self.n, self.nb, self.nranks, self.rank = n, nb, nranks, rank
        opts.setdefault("executor", EXEC_SCHEDULER)
        self.h = chol_plan_dist(n, nb, nranks, rank, **opts)
        if allgather is not None:
            chol_dist_connect(self.h, allgather(chol_dist_export(self.h)))

    @staticmethod
    def connect_local(plans: list) -> None:
        blobs = [chol_dist_export(p.h) for p in plans]
        for p in plans:
            chol_dist_connect(p.h, blobs)

    def close(self):
        if self.h:
            chol_destroy(self.h)
            self.h = 0

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


class Plan:
    """RAII wrapper: ``with Plan(n, nb, executor=EXEC_HOST) as p: info = p.factor(A, L)``."""

    def __init__(self, n: int, nb: int, ngpus: int = 1, **opts):
        self.n, self.nb = n, nb
        self.h = chol_plan_ex(n, nb, ngpus, **opts)

    def factor(self, A, L=None, lda: int | None = None, ldl: int | None = None) -> int:
        L = A if L is None else L
        return chol_factor(self.h, A, lda or self.n, L, ldl or self.n)

    def solve(self, B, ldb: int | None = None) -> None:
        """A X = B in place (B: n x nrhs row-major, host or device) with this plan's factor."""
        nrhs = 1 if len(B.shape) == 1 else B.shape[1]
        chol_solve(self.h, B, ldb or nrhs, nrhs)

    def close(self):
        if self.h:
            chol_destroy(self.h)
            self.h = 0

    def __enter__(self):
        return self

    def __exit__(self, *a):
        self.close()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass
