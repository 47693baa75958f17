// CTA-level tile operations of the tiled Cholesky (Algorithm 1;
// kernels L196-208), written once as __device__ functions and used by both the
// host-sequenced kernels and the persistent scheduler kernel.
//
// Tile store: N(N+1)/2 row-major nb x nb FP64 tiles, tile (i,j), i >= j, at index
// i(i+1)/2 + j.  One 3-D TMA map covers the whole store:
// dims {nb, nb, ntiles}, box {16, BS, 1}, 128-byte swizzle, so any BS-row x 16-column
// slab of any tile lands in shared memory with one cp.async.bulk.tensor.
//
// CTA shape: 8 compute warps (2 x 4 warp grid, warp tile BS/2 x BS/4, FP64 DMMA
// m8n8k4 with register accumulators) + 1 producer warp that issues TMA into a
// kStages-deep mbarrier ring.  Sub-task granularity is a BS x BS block (BS = 96 at
// nb = 960, so a GEMM task is 100 CTA sub-tasks of 96 x 96 x 960).
#pragma once
#include "dev_common.cuh"
#include "taskid.h"

namespace chol {

constexpr int kComputeWarps = 8;
constexpr int kComputeThreads = kComputeWarps * 32;
constexpr int kThreads = kComputeThreads + 32;  // + producer warp
constexpr int kStages = 4;
constexpr int BK = 16;  // doubles per TMA box row (128 bytes)
constexpr int kBarCompute = 1;  // named barrier id: compute warps only
constexpr int kBarAll = 2;      // named barrier id: all warps


template <int BS>
struct Cfg {
  static constexpr int WM = BS / 2, WN = BS / 4;  // warp tile
  static constexpr int MI = WM / 8, NI = WN / 8;  // m8n8 blocks per warp
  static constexpr int kOpBytes = BS * BK * 8;    // one operand, one stage
  static constexpr int kPipeBytes = kStages * 2 * kOpBytes;
  static constexpr int kPitch = BS + 2;            // doubles; keeps double2 alignment
  static constexpr int kBufBytes = BS * kPitch * 8;
  static constexpr int kSmemBytes = kPipeBytes + kBufBytes + 2 * kStages * 8 + 1024;
  static constexpr int RW = BS / kComputeWarps;    // rows per warp in the solves
  static constexpr int CPL = BS / 32;              // columns per lane in the solves
  static_assert(BS % 32 == 0 && WM % 8 == 0 && WN % 8 == 0, "tile shape");
  static_assert(kBufBytes <= kPipeBytes, "solve buffer aliases the pipeline ring");
};

// Per-CTA state: smem carve-up + TMA pipeline position.  Producer and consumers
// walk the same stage sequence, so one counter describes both.
template <int BS>
struct Ctx {
  const CUtensorMap* map;
  double* tiles;
  int nb, N;
  char* pipe;      // kStages x {A, B} operand buffers (1024-aligned)
  double* buf;     // BS x kPitch solve/factor buffer (aliases pipe)
  double* lbuf;    // BS x kPitch (transposed L block)
  uint64_t* full;  // kStages
  uint64_t* empty; // kStages
  uint32_t it;     // stages consumed so far
  int warp, lane;

  __device__ double* tile(int i, int j) const { return tiles + tile_index(i, j) * (int64_t)nb * nb; }
  __device__ bool producer() const { return warp == kComputeWarps; }
};

template <int BS>
__device__ __forceinline__ Ctx<BS> make_ctx(const CUtensorMap* map, double* tiles, int nb, int N) {
  extern __shared__ __align__(1024) char smem_raw[];
  using C = Cfg<BS>;
  Ctx<BS> c;
  char* base = reinterpret_cast<char*>((reinterpret_cast<uintptr_t>(smem_raw) + 1023) & ~uintptr_t(1023));
  c.map = map;
  c.tiles = tiles;
  c.nb = nb;
  c.N = N;
  c.pipe = base;
  c.buf = reinterpret_cast<double*>(base);
  c.lbuf = reinterpret_cast<double*>(base + C::kPipeBytes);
  c.full = reinterpret_cast<uint64_t*>(base + C::kPipeBytes + C::kBufBytes);
  c.empty = c.full + kStages;
  c.it = 0;
  c.warp = threadIdx.x >> 5;
  c.lane = threadIdx.x & 31;
  if (threadIdx.x == 0) {
    for (int s = 0; s < kStages; ++s) {
      mbar_init(&c.full[s], 1);
      mbar_init(&c.empty[s], kComputeWarps);
    }
    fence_mbar_init();
  }
  if (c.producer() && c.lane == 0) tma_prefetch_desc(map);
  __syncthreads();
  return c;
}

template <int BS>
using Acc = double[Cfg<BS>::MI][Cfg<BS>::NI][2];

// acc = A[ra:ra+BS, kbeg:kend] * B[rb:rb+BS, kbeg:kend]^T with A = tile ta, B = tile tb
// (tile-store indices), "NT" form: both operands K-contiguous (row-major tiles).
// kbeg, kend multiples of BK.  Called by all warps of the CTA.
template <int BS>
__device__ __forceinline__ void gemm_mainloop(Ctx<BS>& c, int64_t ta, int ra, int64_t tb, int rb, int kbeg,
                                              int kend, Acc<BS>& acc) {
  using C = Cfg<BS>;
  const int nst = (kend - kbeg) / BK;
  if (c.producer()) {
    if (c.lane == 0) {
      fence_proxy_async();  // operands may have been written by generic stores (this or other SMs)
      for (int s = 0; s < nst; ++s) {
        const uint32_t q = c.it + s, st = q % kStages, ph = (q / kStages) & 1;
        mbar_wait(&c.empty[st], ph ^ 1);
        mbar_arrive_expect_tx(&c.full[st], 2 * C::kOpBytes);
        char* sa = c.pipe + st * 2 * C::kOpBytes;
        tma_load_3d(sa, c.map, &c.full[st], kbeg + s * BK, ra, (int)ta);
        tma_load_3d(sa + C::kOpBytes, c.map, &c.full[st], kbeg + s * BK, rb, (int)tb);
      }
    }
  } else {
#pragma unroll
    for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
      for (int ni = 0; ni < C::NI; ++ni) acc[mi][ni][0] = acc[mi][ni][1] = 0.0;
    const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
    // threadIdx.y is 0 (1-D blocks) but unknown to the compiler: used to make the
    // stage release depend on every shared load of the stage (see below).
    const uint32_t rt_zero = threadIdx.y;
    for (int s = 0; s < nst; ++s) {
      const uint32_t q = c.it + s, st = q % kStages, ph = (q / kStages) & 1;
      mbar_wait(&c.full[st], ph);
      const uint32_t As = smem_u32(c.pipe) + st * 2 * C::kOpBytes + (wm * C::WM + g) * 128;
      const uint32_t Bs = smem_u32(c.pipe) + st * 2 * C::kOpBytes + C::kOpBytes + (wn * C::WN + g) * 128;
      uint32_t dep = 0;
#pragma unroll
      for (int h = 0; h < 2; ++h) {
        // 128B swizzle: 16-byte chunk index ^= (row & 7); rows here are 8-aligned + g.
        const int chunk = ((h * 4 + t) ^ g) << 4;
        double2 af[C::MI], bf[C::NI];
#pragma unroll
        for (int mi = 0; mi < C::MI; ++mi) af[mi] = lds128(As + mi * 8 * 128 + chunk);
#pragma unroll
        for (int ni = 0; ni < C::NI; ++ni) bf[ni] = lds128(Bs + ni * 8 * 128 + chunk);
#pragma unroll
        for (int mi = 0; mi < C::MI; ++mi) dep ^= __double2loint(af[mi].x);
#pragma unroll
        for (int ni = 0; ni < C::NI; ++ni) dep ^= __double2loint(bf[ni].x);
        // k-permutation: thread t holds k = 8h+2t (x) and 8h+2t+1 (y) for both operands.
#pragma unroll
        for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
          for (int ni = 0; ni < C::NI; ++ni) dmma884(acc[mi][ni][0], acc[mi][ni][1], af[mi].x, bf[ni].x);
#pragma unroll
        for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
          for (int ni = 0; ni < C::NI; ++ni) dmma884(acc[mi][ni][0], acc[mi][ni][1], af[mi].y, bf[ni].y);
      }
      // Hand the stage back to the producer only once every ld.shared of it has
      // returned: the arrive is predicated on a value derived from all loaded
      // registers (lane 0 arrives), so it cannot issue before the loads complete
      // and a TMA refill can never overwrite data a lane has not read yet.
      __syncwarp();
      if (c.lane == (int)(dep & rt_zero)) mbar_arrive(&c.empty[st]);
    }
  }
  c.it += nst;
}

// C[0:BS, 0:BS] -= acc for the BS x BS block at Cblk (leading dimension ldc).
// lower_only: diagonal block of a diagonal tile -- only r >= c is written (SYRK, L207-208).
template <int BS>
__device__ __forceinline__ void epi_sub_global(const Ctx<BS>& c, const Acc<BS>& acc, double* Cblk, int ldc,
                                               bool lower_only) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      const int r = wm * C::WM + mi * 8 + g, cc = wn * C::WN + ni * 8 + 2 * t;
      double2* p = reinterpret_cast<double2*>(Cblk + (int64_t)r * ldc + cc);
      double2 v = __ldcg(p);
      v.x -= acc[mi][ni][0];
      v.y -= acc[mi][ni][1];
      if (!lower_only) {
        __stcg(p, v);
      } else {
        if (cc <= r) __stcg(&p->x, v.x);
        if (cc + 1 <= r) __stcg(&p->y, v.y);
      }
    }
}

// X <- (X - acc) * Ld^{-T} for one BS x BS block X (ld ldx) against the lower
// triangular BS x BS diagonal block Ld (ld ldl): the in-block part of TRSM
// (L200-202), forward substitution x_c = (b_c - sum_{m<c} x_m L[c][m]) / L[c][c]
// per row, right-looking inside the block.  Rows are independent, so each
// compute warp owns BS/8 rows in registers (columns split over lanes) and the
// only communication is a warp shuffle of x_c.  Compute warps only; ends with a
// compute-warp barrier.  has_acc = false: acc is ignored (treated as zero).
template <int BS>
__device__ __forceinline__ void solve_block(const Ctx<BS>& c, const Acc<BS>& acc, bool has_acc, double* X, int ldx,
                                            const double* Ld, int ldl) {
  using C = Cfg<BS>;
  const int tid = threadIdx.x;
  // buf aliases the TMA ring: every compute warp must be done reading its last stage.
  bar_sync(kBarCompute, kComputeThreads);
  // 1. buf = X - acc (fragment layout), lbuf = Ld^T (lower part).
  {
    const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
#pragma unroll
    for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
      for (int ni = 0; ni < C::NI; ++ni) {
        const int r = wm * C::WM + mi * 8 + g, cc = wn * C::WN + ni * 8 + 2 * t;
        double2 v = __ldcg(reinterpret_cast<const double2*>(X + (int64_t)r * ldx + cc));
        if (has_acc) {
          v.x -= acc[mi][ni][0];
          v.y -= acc[mi][ni][1];
        }
        *reinterpret_cast<double2*>(c.buf + r * C::kPitch + cc) = v;
      }
    for (int idx = tid; idx < BS * BS; idx += kComputeThreads) {
      const int r = idx / BS, cc = idx - r * BS;
      if (cc <= r) c.lbuf[cc * C::kPitch + r] = __ldcg(Ld + (int64_t)r * ldl + cc);
    }
  }
  bar_sync(kBarCompute, kComputeThreads);
  // 2. per-warp substitution on BS/8 rows held in registers.
  double x[C::RW][C::CPL];
  const int r0 = c.warp * C::RW, lane = c.lane;
#pragma unroll
  for (int q = 0; q < C::RW; ++q)
#pragma unroll
    for (int s = 0; s < C::CPL; ++s) x[q][s] = c.buf[(r0 + q) * C::kPitch + s * 32 + lane];
#pragma unroll
  for (int s = 0; s < C::CPL; ++s) {
    for (int cl = 0; cl < 32; ++cl) {
      const int ci = s * 32 + cl;
      const double* lrow = c.lbuf + ci * C::kPitch;  // lrow[c'] = L[c'][ci]
      const double rd = 1.0 / lrow[ci];
      double lc[C::CPL];
#pragma unroll
      for (int s2 = 0; s2 < C::CPL; ++s2) lc[s2] = (s2 >= s) ? lrow[s2 * 32 + lane] : 0.0;
#pragma unroll
      for (int q = 0; q < C::RW; ++q) {
        const double v = __shfl_sync(0xffffffffu, x[q][s], cl) * rd;
        if (lane == cl) x[q][s] = v;
#pragma unroll
        for (int s2 = s; s2 < C::CPL; ++s2)
          if (s2 * 32 + lane > ci) x[q][s2] = fma(-v, lc[s2], x[q][s2]);
      }
    }
  }
  // 3. write the solved rows back (coalesced).
#pragma unroll
  for (int q = 0; q < C::RW; ++q)
#pragma unroll
    for (int s = 0; s < C::CPL; ++s) __stcg(X + (int64_t)(r0 + q) * ldx + s * 32 + lane, x[q][s]);
  bar_sync(kBarCompute, kComputeThreads);
}

// Unblocked Cholesky of the BS x BS diagonal block A (ld lda), lower, in shared
// memory (POTRF, L196-199).  Right-looking column algorithm; on a pivot !(d > 0)
// records info = col0 + c + 1 with atomicMin (LAPACK convention, reading R6).
// Compute warps only.
template <int BS>
__device__ __forceinline__ void potf2_block(const Ctx<BS>& c, double* A, int lda, int col0, int* info) {
  using C = Cfg<BS>;
  const int tid = threadIdx.x;
  double* a = c.buf;
  bar_sync(kBarCompute, kComputeThreads);  // buf aliases the TMA ring
  for (int idx = tid; idx < BS * BS; idx += kComputeThreads) {
    const int r = idx / BS, cc = idx - r * BS;
    if (cc <= r) a[r * C::kPitch + cc] = __ldcg(A + (int64_t)r * lda + cc);
  }
  bar_sync(kBarCompute, kComputeThreads);
  for (int j = 0; j < BS; ++j) {
    const double d = a[j * C::kPitch + j];
    const double ljj = sqrt(d);
    if (tid == 0 && !(d > 0.0)) atomicMin(info, col0 + j + 1);
    if (tid < BS - 1 - j) {
      const int r = j + 1 + tid;
      a[r * C::kPitch + j] = a[r * C::kPitch + j] / ljj;
    }
    bar_sync(kBarCompute, kComputeThreads);
    if (tid == 0) a[j * C::kPitch + j] = ljj;
    const int m = BS - 1 - j;
    for (int idx = tid; idx < m * m; idx += kComputeThreads) {
      const int rr = idx / m, cc = idx - rr * m;
      if (cc <= rr) {
        const int r = j + 1 + rr, col = j + 1 + cc;
        a[r * C::kPitch + col] = fma(-a[r * C::kPitch + j], a[col * C::kPitch + j], a[r * C::kPitch + col]);
      }
    }
    bar_sync(kBarCompute, kComputeThreads);
  }
  for (int idx = tid; idx < BS * BS; idx += kComputeThreads) {
    const int r = idx / BS, cc = idx - r * BS;
    if (cc <= r) __stcg(A + (int64_t)r * lda + cc, a[r * C::kPitch + cc]);
  }
}

// ------------------------------------------------------------------ sub-tasks
// Each is executed by all warps of one CTA.  Sub-task granularity: a BS x BS
// block (GEMM / SYRK / POTRF-inner), a BS-row slab (TRSM).

// GEMM_i_j_k sub-task (bm, bn):  A_ij[bm, bn] -= L_ik[bm, :] L_jk[bn, :]^T   (L203-206)
// SYRK_j_k  sub-task (bm >= bn): the same with i = j, lower part only      (L207-208)
template <int BS>
__device__ __forceinline__ void sub_update(Ctx<BS>& c, int i, int j, int k, int bm, int bn) {
  Acc<BS> acc;
  gemm_mainloop(c, tile_index(i, k), bm * BS, tile_index(j, k), bn * BS, 0, c.nb, acc);
  if (!c.producer())
    epi_sub_global(c, acc, c.tile(i, j) + (int64_t)bm * BS * c.nb + bn * BS, c.nb, i == j && bm == bn);
}

// TRSM_i_k sub-task = row slab `slab` of A_ik:  X <- X L_kk^{-T}  (L200-202),
// left-looking over BS-column blocks: X[:, cb] = (X[:, cb] - X[:, :cb] L[cb, :cb]^T) L[cb, cb]^{-T}.
template <int BS>
__device__ __forceinline__ void sub_trsm(Ctx<BS>& c, int i, int k, int slab) {
  const int nbb = c.nb / BS;
  double* X = c.tile(i, k) + (int64_t)slab * BS * c.nb;
  const double* L = c.tile(k, k);
  for (int cb = 0; cb < nbb; ++cb) {
    Acc<BS> acc;
    if (cb > 0) gemm_mainloop(c, tile_index(i, k), slab * BS, tile_index(k, k), cb * BS, 0, cb * BS, acc);
    if (!c.producer()) {
      solve_block(c, acc, cb > 0, X + cb * BS, c.nb, L + (int64_t)cb * BS * c.nb + cb * BS, c.nb);
      // X[:, cb] (generic stores) is read by TMA in the next block: complete the stores
      // at L2 (gpu-scope fence), then order them before async-proxy accesses.
      __threadfence();
      fence_proxy_async();
    }
    bar_sync(kBarAll, kThreads);
  }
}

// POTRF_k, inner step b (nested tiled Cholesky of the diagonal tile with block BS):
//   potf2 of block (b, b)
template <int BS>
__device__ __forceinline__ void sub_potrf_diag(Ctx<BS>& c, int k, int b, int* info) {
  if (!c.producer()) {
    double* A = c.tile(k, k) + (int64_t)b * BS * c.nb + b * BS;
    potf2_block(c, A, c.nb, k * c.nb + b * BS, info);
  }
}
//   block (r, b), r > b:  X <- X L_bb^{-T}
template <int BS>
__device__ __forceinline__ void sub_potrf_panel(Ctx<BS>& c, int k, int b, int r) {
  if (!c.producer()) {
    double* T = c.tile(k, k);
    Acc<BS> acc;
    solve_block(c, acc, false, T + (int64_t)r * BS * c.nb + b * BS, c.nb, T + (int64_t)b * BS * c.nb + b * BS, c.nb);
  }
}
//   block (r, q), b < q <= r:  A[r, q] -= L[r, b] L[q, b]^T   (K = BS)
template <int BS>
__device__ __forceinline__ void sub_potrf_update(Ctx<BS>& c, int k, int b, int r, int q) {
  Acc<BS> acc;
  const int64_t t = tile_index(k, k);
  gemm_mainloop(c, t, r * BS, t, q * BS, b * BS, (b + 1) * BS, acc);
  if (!c.producer()) epi_sub_global(c, acc, c.tile(k, k) + (int64_t)r * BS * c.nb + q * BS, c.nb, r == q);
}

}  // namespace chol
