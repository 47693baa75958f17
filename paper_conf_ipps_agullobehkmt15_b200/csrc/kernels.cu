// Host-sequenced executor kernels (CHOL_EXEC_HOST), layout / generator kernels and
// their launchers.  Each kernel runs one sub-task per CTA via the tile ops in
// tile_ops.cuh; the persistent scheduler (scheduler.cu) runs the same tile ops.
#include <climits>
#include <cstdio>

#include "kernels.h"
#include "taskid.h"
#include "tile_ops.cuh"

namespace chol {

// ------------------------------------------------------------------ trace helpers
__device__ __forceinline__ uint64_t trace_now(const StepParams& p) {
  return p.tr_base ? globaltimer_ns() - *p.tr_base : 0;
}
__device__ __forceinline__ void trace_record(const StepParams& p, int64_t task, uint64_t t_start) {
  if (!p.tr_t0) return;
  __syncthreads();
  if (threadIdx.x == 0) {
    const uint64_t t_end = globaltimer_ns() - *p.tr_base;
    atomicMin(reinterpret_cast<unsigned long long*>(p.tr_t0 + task), (unsigned long long)t_start);
    atomicMax(reinterpret_cast<unsigned long long*>(p.tr_t1 + task), (unsigned long long)((t_end << 16) | smid()));
  }
}

// ------------------------------------------------------------------ POTRF (nested, block BS)
template <int BS>
__global__ void __launch_bounds__(kThreads, 1) k_potrf_diag(const __grid_constant__ CUtensorMap map, StepParams p) {
  const uint64_t t0 = trace_now(p);
  auto c = make_ctx<BS>(&map, p.tiles, p.nb, p.N);
  const int k = p.k + blockIdx.y;
  sub_potrf_diag(c, k, p.b, p.info);
  trace_record(p, id_potrf(p.N, k), t0);
}

template <int BS>
__global__ void __launch_bounds__(kThreads, 1) k_potrf_panel(const __grid_constant__ CUtensorMap map, StepParams p) {
  const uint64_t t0 = trace_now(p);
  auto c = make_ctx<BS>(&map, p.tiles, p.nb, p.N);
  const int k = p.k + blockIdx.y;
  sub_potrf_panel(c, k, p.b, p.b + 1 + blockIdx.x);
  trace_record(p, id_potrf(p.N, k), t0);
}

template <int BS>
__global__ void __launch_bounds__(kThreads, 1) k_potrf_update(const __grid_constant__ CUtensorMap map, StepParams p) {
  const uint64_t t0 = trace_now(p);
  auto c = make_ctx<BS>(&map, p.tiles, p.nb, p.N);
  const int k = p.k + blockIdx.y;
  const int nbb = p.nb / BS, m = nbb - 1 - p.b;
  // blockIdx.x enumerates (r, q), b < q <= r < nbb, row by row
  int rem = blockIdx.x, rr = 0;
  while (rem > rr) {
    rem -= rr + 1;
    ++rr;
  }
  (void)m;
  sub_potrf_update(c, k, p.b, p.b + 1 + rr, p.b + 1 + rem);
  trace_record(p, id_potrf(p.N, k), t0);
}

// ------------------------------------------------------------------ TRSM batch
// inverses of the diagonal blocks of L_kk (blockIdx.x = b), for the inverse-form slabs
template <int BS>
__global__ void __launch_bounds__(kThreads, 1) k_inv(const __grid_constant__ CUtensorMap map, StepParams p) {
  auto c = make_ctx<BS>(&map, p.tiles, p.nb, p.N);
  const int nbb = p.nb / BS, b = blockIdx.x;
  inv_block(c, c.tile(p.k, p.k) + (int64_t)b * BS * p.nb + b * BS, p.nb, p.dinv + ((int64_t)p.k * nbb + b) * BS * BS);
}

// blockIdx.x = task * nbb + slab, task -> i = i0 + task (all with the same k)
template <int BS>
__global__ void __launch_bounds__(kThreads, 1) k_trsm(const __grid_constant__ CUtensorMap map,
                                                      const __grid_constant__ CUtensorMap dmap, StepParams p) {
  const uint64_t t0 = trace_now(p);
  auto c = make_ctx<BS>(&map, p.tiles, p.nb, p.N);
  const int nbb = p.nb / BS;
  const int i = p.i0 + blockIdx.x / nbb, slab = blockIdx.x % nbb;
  sub_trsm_inv(c, &dmap, i, p.k, slab);
  trace_record(p, id_trsm(p.N, i, p.k), t0);
}

// ------------------------------------------------------------------ SYRK / GEMM batch
// mode 0: all SYRK+GEMM of step k;  1: the single task (i0, j0, k);
// mode 2: only the GEMMs of step k; 3: only the SYRKs of step k.
template <int BS>
__global__ void __launch_bounds__(kThreads, 1) k_update(const __grid_constant__ CUtensorMap map, StepParams p) {
  const uint64_t t0 = trace_now(p);
  const int nbb = p.nb / BS;
  const int task = blockIdx.x / (nbb * nbb), sub = blockIdx.x % (nbb * nbb);
  const int bm = sub / nbb, bn = sub % nbb;
  int i, j;
  const int k = p.k, m = p.N - 1 - k;
  if (p.mode == 1) {
    i = p.i0;
    j = p.j0;
  } else if (p.mode == 3) {
    i = j = k + 1 + task;
  } else if (p.mode == 2) {
    // (j, i) with k < j < i < N, row by row of j
    int rem = task, jj = 0;
    while (rem >= m - 1 - jj) {
      rem -= m - 1 - jj;
      ++jj;
    }
    j = k + 1 + jj;
    i = j + 1 + rem;
  } else {
    // (j, i) with k < j <= i < N, row by row of j (Algorithm 1 order)
    int rem = task, jj = 0;
    while (rem >= m - jj) {
      rem -= m - jj;
      ++jj;
    }
    j = k + 1 + jj;
    i = j + rem;
  }
  if (i == j && bn > bm) return;  // SYRK: strictly-upper blocks are not needed
  auto c = make_ctx<BS>(&map, p.tiles, p.nb, p.N);
  sub_update(c, i, j, k, bm, bn);
  trace_record(p, i == j ? id_syrk(p.N, j, k) : id_gemm(p.N, i, j, k), t0);
}

// ------------------------------------------------------------------ small kernels
__global__ void k_stamp(uint64_t* base) { *base = globaltimer_ns(); }

__global__ void k_init_info(int* info) { *info = INT_MAX; }

// mark every input tile as arrived (factorizations whose input is already resident)
__global__ void k_fill_flags(int* flags, int64_t n, int value) {
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x)
    flags[i] = value;
}

// zero the strictly upper triangle of every diagonal tile
// slots: store slots of the diagonal tiles to clean (null: tile k at tile_index(k, k))
__global__ void k_zero_upper_diag(double* tiles, int nb, int N, const int* slots) {
  const int k = blockIdx.y;
  double* T = tiles + (slots ? (int64_t)slots[k] : tile_index(k, k)) * (int64_t)nb * nb;
  for (int64_t idx = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; idx < (int64_t)nb * nb;
       idx += (int64_t)gridDim.x * blockDim.x) {
    const int r = (int)(idx / nb), c = (int)(idx % nb);
    if (c > r) T[idx] = 0.0;
  }
}

// ------------------------------------------------------------------ generator
// Counter-based synthetic SPD inputs; an independent
// implementation of the recipe the Python side (spdgen/) implements.
__device__ __forceinline__ uint64_t splitmix64(uint64_t z) {
  z += 0x9E3779B97F4A7C15ull;
  z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
  return z ^ (z >> 31);
}
constexpr uint64_t kIntSalt = 0xD1B54A32D192ED03ull;
constexpr int kBW = 3;

// L0[x][x-o] of the integer family
__device__ __forceinline__ int64_t l0_band(uint64_t seed, int64_t n, int64_t x, int o) {
  if (x - o < 0) return 0;
  const uint64_t key = (seed ^ kIntSalt) * 0x9E3779B97F4A7C15ull + (uint64_t)x * (uint64_t)n + (uint64_t)(x - o);
  const uint64_t z = splitmix64(key);
  if (o == 0) {
    const int sel = (int)((z >> 32) % 3);
    return sel == 0 ? 1 : (sel == 1 ? 2 : 4);
  }
  const int top = (int)(z >> 61);
  return top < 2 ? -1 : (top < 4 ? 1 : 0);
}

// slot_tile: tile index held by each generated store slot (null: slot == tile index)
__global__ void k_generate(double* tiles, int64_t n, int nb, int N, uint64_t seed, int family, int64_t t_off,
                           const int* slot_tile) {
  const int64_t slot = t_off + blockIdx.y;
  const int64_t t = slot_tile ? (int64_t)slot_tile[slot] : slot;  // tile index
  // decode t -> (ti, tj), ti >= tj
  int ti = (int)((sqrt(8.0 * (double)t + 1.0) - 1.0) / 2.0);
  while ((int64_t)ti * (ti + 1) / 2 > t) --ti;
  while ((int64_t)(ti + 1) * (ti + 2) / 2 <= t) ++ti;
  const int tj = (int)(t - (int64_t)ti * (ti + 1) / 2);
  double* T = tiles + slot * (int64_t)nb * nb;
  for (int64_t idx = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; idx < (int64_t)nb * nb;
       idx += (int64_t)gridDim.x * blockDim.x) {
    const int64_t r = idx / nb, c = idx % nb;
    const int64_t gi = (int64_t)ti * nb + r, gj = (int64_t)tj * nb + c;
    const int64_t hi = gi > gj ? gi : gj, lo = gi > gj ? gj : gi;
    double v;
    if (family == 0) {
      const uint64_t key = seed * 0x9E3779B97F4A7C15ull + (uint64_t)hi * (uint64_t)n + (uint64_t)lo;
      v = (double)(splitmix64(key) >> 11) * 0x1.0p-53 - 0.5;
      if (hi == lo) v += (double)n;
    } else {
      const int o = (int)(hi - lo);
      int64_t acc = 0;
      if (o <= kBW)
        for (int q = o; q <= kBW; ++q) acc += l0_band(seed, n, hi, q) * l0_band(seed, n, lo, q - o);
      v = (double)acc;
    }
    T[idx] = v;
  }
}

// ------------------------------------------------------------------ launchers
// cudaFuncSetAttribute acts on the current device's context: set it on every call (a
// plan on another device, or another thread, must not find it skipped); it is cheap.
template <int BS>
static cudaError_t set_attrs() {
  const int bytes = Cfg<BS>::kSmemBytes;
  cudaError_t e;
  if ((e = cudaFuncSetAttribute(k_potrf_diag<BS>, cudaFuncAttributeMaxDynamicSharedMemorySize, bytes))) return e;
  if ((e = cudaFuncSetAttribute(k_potrf_panel<BS>, cudaFuncAttributeMaxDynamicSharedMemorySize, bytes))) return e;
  if ((e = cudaFuncSetAttribute(k_potrf_update<BS>, cudaFuncAttributeMaxDynamicSharedMemorySize, bytes))) return e;
  if ((e = cudaFuncSetAttribute(k_trsm<BS>, cudaFuncAttributeMaxDynamicSharedMemorySize, bytes))) return e;
  if ((e = cudaFuncSetAttribute(k_inv<BS>, cudaFuncAttributeMaxDynamicSharedMemorySize, bytes))) return e;
  if ((e = cudaFuncSetAttribute(k_update<BS>, cudaFuncAttributeMaxDynamicSharedMemorySize, bytes))) return e;
  return cudaSuccess;
}

template <int BS>
static int launch_potrf_t(const CUtensorMap& map, StepParams p, int count, cudaStream_t s, int* nlaunch) {
  const int nbb = p.nb / BS, smem = Cfg<BS>::kSmemBytes;
  for (int b = 0; b < nbb; ++b) {
    p.b = b;
    k_potrf_diag<BS><<<dim3(1, count), kThreads, smem, s>>>(map, p);
    ++*nlaunch;
    const int m = nbb - 1 - b;
    if (m > 0) {
      k_potrf_panel<BS><<<dim3(m, count), kThreads, smem, s>>>(map, p);
      k_potrf_update<BS><<<dim3(m * (m + 1) / 2, count), kThreads, smem, s>>>(map, p);
      *nlaunch += 2;
    }
  }
  return 0;
}

template <int BS>
static int launch_trsm_t(const CUtensorMap& map, const CUtensorMap& dmap, StepParams p, int count, cudaStream_t s,
                         int* nlaunch) {
  const int nbb = p.nb / BS;
  k_inv<BS><<<nbb, kThreads, Cfg<BS>::kSmemBytes, s>>>(map, p);
  k_trsm<BS><<<count * nbb, kThreads, Cfg<BS>::kSmemBytes, s>>>(map, dmap, p);
  *nlaunch += 2;
  return 0;
}

template <int BS>
static int launch_update_t(const CUtensorMap& map, StepParams p, int ntask, cudaStream_t s, int* nlaunch) {
  const int nbb = p.nb / BS;
  k_update<BS><<<ntask * nbb * nbb, kThreads, Cfg<BS>::kSmemBytes, s>>>(map, p);
  ++*nlaunch;
  return 0;
}

#define CHOL_DISPATCH(bs, call)            \
  switch (bs) {                            \
    case 96: call(96); break;              \
    case 64: call(64); break;              \
    case 32: call(32); break;              \
    default: return cudaErrorInvalidValue; \
  }

cudaError_t prepare_kernels(int bs) {
#define PREP(B) return set_attrs<B>()
  CHOL_DISPATCH(bs, PREP)
#undef PREP
  return cudaSuccess;
}

int smem_bytes(int bs) {
  switch (bs) {
    case 96: return Cfg<96>::kSmemBytes;
    case 64: return Cfg<64>::kSmemBytes;
    case 32: return Cfg<32>::kSmemBytes;
  }
  return 0;
}

cudaError_t launch_potrf(int bs, const CUtensorMap& map, const StepParams& p, int count, cudaStream_t s, int* nl) {
#define L(B) launch_potrf_t<B>(map, p, count, s, nl)
  CHOL_DISPATCH(bs, L)
#undef L
  return cudaGetLastError();
}
cudaError_t launch_trsm(int bs, const CUtensorMap& map, const CUtensorMap& dmap, const StepParams& p, int count,
                        cudaStream_t s, int* nl) {
#define L(B) launch_trsm_t<B>(map, dmap, p, count, s, nl)
  CHOL_DISPATCH(bs, L)
#undef L
  return cudaGetLastError();
}
cudaError_t launch_update(int bs, const CUtensorMap& map, const StepParams& p, int ntask, cudaStream_t s, int* nl) {
#define L(B) launch_update_t<B>(map, p, ntask, s, nl)
  CHOL_DISPATCH(bs, L)
#undef L
  return cudaGetLastError();
}

cudaError_t launch_stamp(uint64_t* base, cudaStream_t s) {
  k_stamp<<<1, 1, 0, s>>>(base);
  return cudaGetLastError();
}
cudaError_t launch_fill_flags(int* flags, int64_t n, int value, cudaStream_t s) {
  k_fill_flags<<<(unsigned)((n + 255) / 256 < 1024 ? (n + 255) / 256 : 1024), 256, 0, s>>>(flags, n, value);
  return cudaGetLastError();
}
cudaError_t launch_init_info(int* info, cudaStream_t s) {
  k_init_info<<<1, 1, 0, s>>>(info);
  return cudaGetLastError();
}
cudaError_t launch_zero_upper_diag(double* tiles, int nb, int N, cudaStream_t s, const int* slots, int count) {
  if (count == 0) return cudaSuccess;
  k_zero_upper_diag<<<dim3(64, slots ? count : N), 256, 0, s>>>(tiles, nb, N, slots);
  return cudaGetLastError();
}
cudaError_t launch_generate(double* tiles, int64_t n, int nb, int N, uint64_t seed, int family, cudaStream_t s,
                            const int* slot_tile, int64_t nslots) {
  const int64_t ntiles = slot_tile ? nslots : (int64_t)N * (N + 1) / 2;
  for (int64_t t0 = 0; t0 < ntiles; t0 += 65535) {
    const int64_t cnt = ntiles - t0 < 65535 ? ntiles - t0 : 65535;
    k_generate<<<dim3(64, (unsigned)cnt), 256, 0, s>>>(tiles, n, nb, N, seed, family, t0, slot_tile);
  }
  return cudaGetLastError();
}

}  // namespace chol
