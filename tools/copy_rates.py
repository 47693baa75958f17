"""Host<->device copy rates for the tile layout (cudaMemcpy2DAsync per nb x nb tile from a
row-major pinned matrix) vs one contiguous copy: the e2e path's bandwidth ceiling."""
import sys, time, json
import torch
from cuda.bindings import runtime as rt

n = int(sys.argv[1]) if len(sys.argv) > 1 else 19200
nb = int(sys.argv[2]) if len(sys.argv) > 2 else 960
N = n // nb
nt = N * (N + 1) // 2
A = torch.empty((n, n), dtype=torch.float64, pin_memory=True)
A.fill_(1.0)
d = torch.empty((nt, nb, nb), dtype=torch.float64, device="cuda")
res = {"n": n, "nb": nb, "tile_GB": nt * nb * nb * 8 / 1e9}
for nstreams in (1, 2, 4):
    ss = [rt.cudaStreamCreate()[1] for _ in range(nstreams)]
    for rep in range(2):
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        t = 0
        for i in range(N):
            for j in range(i + 1):
                rt.cudaMemcpy2DAsync(d[t].data_ptr(), nb * 8, A.data_ptr() + (i * nb * n + j * nb) * 8, n * 8,
                                     nb * 8, nb, rt.cudaMemcpyKind.cudaMemcpyHostToDevice, ss[t % nstreams])
                t += 1
        for s in ss:
            rt.cudaStreamSynchronize(s)
        dt = time.perf_counter() - t0
    res[f"h2d_2d_{nstreams}s_GBps"] = round(res["tile_GB"] / dt, 1)
    for rep in range(2):
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        t = 0
        for i in range(N):
            for j in range(i + 1):
                rt.cudaMemcpy2DAsync(A.data_ptr() + (i * nb * n + j * nb) * 8, n * 8, d[t].data_ptr(), nb * 8,
                                     nb * 8, nb, rt.cudaMemcpyKind.cudaMemcpyDeviceToHost, ss[t % nstreams])
                t += 1
        for s in ss:
            rt.cudaStreamSynchronize(s)
        dt = time.perf_counter() - t0
    res[f"d2h_2d_{nstreams}s_GBps"] = round(res["tile_GB"] / dt, 1)
flat = A.view(-1)[: nt * nb * nb]
dflat = d.view(-1)
for rep in range(2):
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    dflat.copy_(flat, non_blocking=True)
    torch.cuda.synchronize()
    dt = time.perf_counter() - t0
res["h2d_flat_GBps"] = round(res["tile_GB"] / dt, 1)
for rep in range(2):
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    flat.copy_(dflat, non_blocking=True)
    torch.cuda.synchronize()
    dt = time.perf_counter() - t0
res["d2h_flat_GBps"] = round(res["tile_GB"] / dt, 1)
# both directions at once
s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()
B = torch.empty_like(flat).pin_memory()
d2 = torch.empty_like(dflat)
torch.cuda.synchronize()
t0 = time.perf_counter()
with torch.cuda.stream(s1):
    dflat.copy_(flat, non_blocking=True)
with torch.cuda.stream(s2):
    B.copy_(d2, non_blocking=True)
torch.cuda.synchronize()
dt = time.perf_counter() - t0
res["duplex_GBps_each"] = round(res["tile_GB"] / dt, 1)
print(json.dumps(res))
