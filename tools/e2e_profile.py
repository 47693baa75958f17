"""End-to-end (host pinned buffers) factorization: wall time, device factor time, and the
scheduler's utilisation timeline while tiles stream in (job trace)."""
import sys, os, json, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import torch
import paper_conf_ipps_agullobehkmt15_b200 as c

n = int(sys.argv[1]) if len(sys.argv) > 1 else 19200
nb = 960
N = n // nb
A_h = torch.empty((n, n), dtype=torch.float64, pin_memory=True)
L_h = torch.empty((n, n), dtype=torch.float64, pin_memory=True)
with c.Plan(n, nb, executor=c.EXEC_SCHEDULER, policy=c.POLICY_CP_PRIORITY, trace=2) as p:
    c.chol_generate(p.h, 0, 0)
    c.chol_gather(p.h, A_h, n)
    walls = []
    for it in range(3):
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        info = c.chol_factor(p.h, A_h, n, L_h, n)
        walls.append(time.perf_counter() - t0)
    tf, tl = c.chol_last_times(p.h)
    jt = c.chol_job_trace(p.h)
    # plain copy rates for reference
    d = torch.empty((N * (N + 1) // 2, nb, nb), dtype=torch.float64, device="cuda")
    src = A_h.view(N, nb, N, nb)
    s = torch.cuda.Stream()
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    with torch.cuda.stream(s):
        t = 0
        for i in range(N):
            for j in range(i + 1):
                d[t].copy_(src[i, :, j, :], non_blocking=True)
                t += 1
    s.synchronize()
    h2d = time.perf_counter() - t0
    t0 = time.perf_counter()
    dst = L_h.view(N, nb, N, nb)
    with torch.cuda.stream(s):
        t = 0
        for i in range(N):
            for j in range(i + 1):
                dst[i, :, j, :].copy_(d[t], non_blocking=True)
                t += 1
    s.synchronize()
    d2h = time.perf_counter() - t0
t0j, t1j = jt[:, 0].astype(np.int64), jt[:, 1].astype(np.int64)
worker = (jt[:, 2] >> np.uint64(32)).astype(np.int64)
W = worker.max() + 1
T0, T1 = t0j.min(), t1j.max()
bins = 20
edges = np.linspace(T0, T1, bins + 1)
util = []
for lo, hi in zip(edges[:-1], edges[1:]):
    ov = np.clip(np.minimum(t1j, hi) - np.maximum(t0j, lo), 0, None).sum()
    util.append(round(float(ov / (W * (hi - lo))), 2))
tile_gb = N * (N + 1) // 2 * nb * nb * 8 / 1e9
print(json.dumps({"n": n, "wall_ms": [round(w * 1e3, 2) for w in walls], "factor_ms": round(tf * 1e3, 2),
                  "layout_ms": round(tl * 1e3, 2), "span_ms": round((T1 - T0) / 1e6, 2),
                  "tile_GB": round(tile_gb, 3), "h2d_ms": round(h2d * 1e3, 2), "h2d_GBps": round(tile_gb / h2d, 1),
                  "d2h_ms": round(d2h * 1e3, 2), "d2h_GBps": round(tile_gb / d2h, 1), "util_timeline": util}))
# arrival as seen by the scheduler: enqueue time of the first-touch task of each tile,
# against the copy order (column 0, then per column j: diagonal tile, tiles below)
ids = {}
for k in range(N):
    ids[c.chol_task_id(N, 0, k, k, k)] = (k, k)
    for i in range(k + 1, N):
        ids[c.chol_task_id(N, 1, i, k, k)] = (i, k)
    for j in range(k + 1, N):
        if k == 0:
            ids[c.chol_task_id(N, 2, j, j, k)] = (j, j)
            for i in range(j + 1, N):
                ids[c.chol_task_id(N, 3, i, j, k)] = (i, j)
order = [(0, 0)] + [(i, 0) for i in range(1, N)]
for j in range(1, N):
    order += [(j, j)] + [(i, j) for i in range(j + 1, N)]
task = (jt[:, 3] & np.uint64(0xffffffff)).astype(np.int64)
tq = jt[:, 4].astype(np.int64)
first_enq = {}
for tid, tile in ids.items():
    m = task == tid
    if m.any():
        first_enq[tile] = (tq[m].min() - T0) / 1e6
pos = [(p, first_enq.get(t)) for p, t in enumerate(order) if t in first_enq]
print(json.dumps({"arrival_seen_ms_by_copy_position": [(p, round(v, 2)) for p, v in pos[::10]],
                  "expected_ms_per_tile_at_53GBps": round(nb * nb * 8 / 53.6e9 * 1e3, 4)}))
