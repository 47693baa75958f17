// CTA-level tile operations of the tiled Cholesky (Algorithm 1;
// kernels L196-208), written once as __device__ functions and used by both the
// host-sequenced kernels and the persistent scheduler kernel.
//
// Tile store: N(N+1)/2 row-major nb x nb FP64 tiles, tile (i,j), i >= j, at index
// i(i+1)/2 + j.  One 3-D TMA map covers the whole store:
// dims {nb, nb, ntiles}, box {16, BS, 1}, 128-byte swizzle, so any BS-row x 16-column
// slab of any tile lands in shared memory with one cp.async.bulk.tensor.
//
// CTA shape: 8 warps (2 x 4 warp grid, warp tile BS/2 x BS/4, FP64 DMMA m8n8k4 with
// register accumulators); thread 0 also issues the TMA loads, kStages-1 stages ahead,
// into a kStages-deep mbarrier ring.  (No dedicated producer warp: 256 threads keep
// the per-thread register budget at 255 -- a 9th warp caps it at 168.)  Sub-task granularity is a BS x BS block (BS = 96 at
// nb = 960, so a GEMM task is 100 CTA sub-tasks of 96 x 96 x 960).
#pragma once
#include "dev_common.cuh"
#include "taskid.h"

namespace chol {

constexpr int kComputeWarps = 8;
constexpr int kComputeThreads = kComputeWarps * 32;
constexpr int kThreads = kComputeThreads;
constexpr int kStages = 5;
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
  static constexpr int kSmemBytes = kPipeBytes + kBufBytes + (2 * kStages + 2) * 8 + 1024;
  static_assert(kBufBytes >= BS * BS * 8, "lbuf holds a TMA-prefetched BS x BS C block");
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
  uint64_t* cbar;  // C-block prefetch (TMA -> lbuf)
  uint32_t it;     // stages consumed so far
  uint32_t cphase; // parity of the next cbar completion
  int warp, lane;

  __device__ double* tile(int i, int j) const { return tiles + tile_index(i, j) * (int64_t)nb * nb; }
  __device__ bool issuer() const { return threadIdx.x == 0; }
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
  c.cbar = c.empty + kStages;
  c.it = 0;
  c.cphase = 0;
  c.warp = threadIdx.x >> 5;
  c.lane = threadIdx.x & 31;
  if (threadIdx.x == 0) {
    for (int s = 0; s < kStages; ++s) {
      mbar_init(&c.full[s], 1);
      mbar_init(&c.empty[s], kComputeWarps);
    }
    mbar_init(c.cbar, 1);
    fence_mbar_init();
  }
  if (c.issuer()) tma_prefetch_desc(map);
  __syncthreads();
  return c;
}

template <int BS>
using Acc = double[Cfg<BS>::MI][Cfg<BS>::NI][2];

// acc = A[ra:ra+BS, kbeg:kend] * B[rb:rb+BS, kbeg:kend]^T with A = tile ta, B = tile tb
// (tile-store indices), "NT" form: both operands K-contiguous (row-major tiles).
// kbeg, kend multiples of BK.  Called by all warps of the CTA.
// Prefetch the BS x BS block (rows r0.., cols c0..) of store tile `tile` into lbuf with
// TMA (BS/16 boxes of BS rows x 128 B, 128B-swizzled), completing on cbar.  Issued by
// thread 0 right after the mainloop prologue so the epilogue's C read overlaps the
// mainloop.
struct CPrefetch {
  int64_t tile;
  int r0, c0;
};

template <int BS>
__device__ __forceinline__ void prefetch_c(Ctx<BS>& c, int64_t tile, int r0, int c0) {
  if (!c.issuer()) return;
  fence_proxy_async();
  mbar_arrive_expect_tx(c.cbar, BS * BS * 8);
  char* dst = reinterpret_cast<char*>(c.lbuf);
#pragma unroll 1
  for (int b = 0; b < BS / 16; ++b) tma_load_3d(dst + b * BS * 128, c.map, c.cbar, c0 + 16 * b, r0, (int)tile);
}

template <int BS>
__device__ __forceinline__ void issue_stage(Ctx<BS>& c, uint32_t q, int64_t ta, int ra, int64_t tb, int rb, int kk) {
  using C = Cfg<BS>;
  const uint32_t st = q % kStages, ph = (q / kStages) & 1;
  mbar_wait(&c.empty[st], ph ^ 1);  // the previous use of this buffer was released by all warps
  mbar_arrive_expect_tx(&c.full[st], 2 * C::kOpBytes);
  char* sa = c.pipe + st * 2 * C::kOpBytes;
  tma_load_3d(sa, c.map, &c.full[st], kk, ra, (int)ta);
  tma_load_3d(sa + C::kOpBytes, c.map, &c.full[st], kk, rb, (int)tb);
}

template <int BS>
__device__ __forceinline__ void gemm_mainloop(Ctx<BS>& c, int64_t ta, int ra, int64_t tb, int rb, int kbeg,
                                              int kend, Acc<BS>& acc, const CPrefetch* cpre = nullptr) {
  using C = Cfg<BS>;
  const int nst = (kend - kbeg) / BK;
  if (c.issuer()) {
    fence_proxy_async();  // operands may have been written by generic stores (this or other SMs)
    const int pre = nst < kStages - 1 ? nst : kStages - 1;
    for (int s = 0; s < pre; ++s) issue_stage(c, c.it + s, ta, ra, tb, rb, kbeg + s * BK);
    if (cpre) prefetch_c(c, cpre->tile, cpre->r0, cpre->c0);
  }
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) acc[mi][ni][0] = acc[mi][ni][1] = 0.0;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  // threadIdx.y is 0 (1-D blocks) but unknown to the compiler: used to make the
  // stage release depend on every shared load of the stage (see below).
  const uint32_t rt_zero = threadIdx.y;
  for (int s = 0; s < nst; ++s) {
    // keep kStages-1 stages in flight: refill the buffer stage s-1 used
    if (c.issuer() && s + kStages - 1 < nst)
      issue_stage(c, c.it + s + kStages - 1, ta, ra, tb, rb, kbeg + (s + kStages - 1) * BK);
    const uint32_t q = c.it + s, st = q % kStages, ph = (q / kStages) & 1;
    mbar_wait(&c.full[st], ph);
    const uint32_t As = smem_u32(c.pipe) + st * 2 * C::kOpBytes + (wm * C::WM + g) * 128;
    const uint32_t Bs = smem_u32(c.pipe) + st * 2 * C::kOpBytes + C::kOpBytes + (wn * C::WN + g) * 128;
    uint32_t dep = 0;
#pragma unroll
    for (int h = 0; h < 2; ++h) {
      // Thread (g, t) reads logical 16-byte chunk 2t + h of its row (k = 4t + 2h, +1):
      // with the 128B swizzle (chunk ^= row & 7) the two rows g, g+1 of one 8-lane
      // phase land on chunks of opposite parity -> conflict-free LDS.128.
      const int chunk = ((2 * t + h) ^ g) << 4;
      double2 af[C::MI], bf[C::NI];
#pragma unroll
      for (int mi = 0; mi < C::MI; ++mi) af[mi] = lds128(As + mi * 8 * 128 + chunk);
#pragma unroll
      for (int ni = 0; ni < C::NI; ++ni) bf[ni] = lds128(Bs + ni * 8 * 128 + chunk);
#pragma unroll
      for (int mi = 0; mi < C::MI; ++mi) dep ^= __double2loint(af[mi].x);
#pragma unroll
      for (int ni = 0; ni < C::NI; ++ni) dep ^= __double2loint(bf[ni].x);
      // k-permutation: thread t holds k = 4t+2h (x) and 4t+2h+1 (y) for both operands.
#pragma unroll
      for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
        for (int ni = 0; ni < C::NI; ++ni) dmma884(acc[mi][ni][0], acc[mi][ni][1], af[mi].x, bf[ni].x);
#pragma unroll
      for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
        for (int ni = 0; ni < C::NI; ++ni) dmma884(acc[mi][ni][0], acc[mi][ni][1], af[mi].y, bf[ni].y);
    }
    // Release the stage only once every ld.shared of it has returned: the arrive is
    // predicated on a value derived from all loaded registers (lane 0 arrives), so it
    // cannot issue before the loads complete and a TMA refill can never overwrite
    // data a lane has not read yet.
    __syncwarp();
    if (c.lane == (int)(dep & rt_zero)) mbar_arrive(&c.empty[st]);
  }
  c.it += nst;
}

// Prefetch the BS x BS block (rows r0.., cols c0..) of store tile `tile` into lbuf with
// TMA (BS/16 boxes of BS rows x 128 B, 128B-swizzled), completing on cbar.  Issued by
// thread 0 at the start of a job so the C read of the epilogue overlaps the mainloop.
// C[0:BS, 0:BS] -= acc for the BS x BS block at Cblk (leading dimension ldc); the old
// C values come from the lbuf prefetch (prefetch_c), results go to global memory.
// lower_only: diagonal block of a diagonal tile -- only r >= c is written (SYRK, L207-208).
template <int BS>
__device__ __forceinline__ void epi_sub_global(Ctx<BS>& c, const Acc<BS>& acc, double* Cblk, int ldc,
                                               bool lower_only) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  mbar_wait(c.cbar, c.cphase);
  c.cphase ^= 1;
  const uint32_t cs = smem_u32(c.lbuf);
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      const int r = wm * C::WM + mi * 8 + g, cc = wn * C::WN + ni * 8 + 2 * t;
      // box cc/16, row r, logical 16-byte chunk (cc%16)/2, 128B swizzle
      const uint32_t addr = cs + (cc >> 4) * (BS * 128) + r * 128 + ((((cc & 15) >> 1) ^ (r & 7)) << 4);
      double2 v = lds128(addr);
      v.x -= acc[mi][ni][0];
      v.y -= acc[mi][ni][1];
      double2* p = reinterpret_cast<double2*>(Cblk + (int64_t)r * ldc + cc);
      if (!lower_only) {
        __stcg(p, v);
      } else {
        if (cc <= r) __stcg(&p->x, v.x);
        if (cc + 1 <= r) __stcg(&p->y, v.y);
      }
    }
}

// D(8x8) -= A(8x8 rows ar.., K=8 at column ak) * B(8x8 rows br.., K=8 at column bk)^T
// on row-major shared-memory operands with pitch P (doubles): two m8n8k4 DMMAs.
// d = {D[g][2t], D[g][2t+1]} fragment.
template <int P>
__device__ __forceinline__ void smem_dmma_sub8(double& d0, double& d1, const double* A, int ar, int ak,
                                               const double* Bm, int br, int bk, int g, int t) {
#pragma unroll
  for (int kk = 0; kk < 8; kk += 4) {
    const double a = -A[(ar + g) * P + ak + kk + t];
    const double bv = Bm[(br + g) * P + bk + kk + t];
    dmma884(d0, d1, a, bv);
  }
}

// X <- (X - acc) * Ld^{-T} for one BS x BS block X (ld ldx) against the lower
// triangular BS x BS diagonal block Ld (ld ldl): the in-block part of TRSM
// (L200-202), forward substitution x_c = (b_c - sum_{m<c} x_m L[c][m]) / L[c][c]
// per row.  Blocked right-looking over 8-column panels: a panel is solved by
// substitution (one thread per row), then the trailing columns are updated with
// FP64 DMMA (X[:, rest] -= X[:, panel] L[rest, panel]^T).  Compute warps only.
// has_acc = false: acc is ignored (treated as zero).
template <int BS>
__device__ __forceinline__ void solve_block(const Ctx<BS>& c, const Acc<BS>& acc, bool has_acc, double* X, int ldx,
                                            const double* Ld, int ldl) {
  using C = Cfg<BS>;
  constexpr int P = C::kPitch;
  const int tid = threadIdx.x, g = c.lane >> 2, t = c.lane & 3;
  double* xb = c.buf;   // X block (aliases the TMA ring)
  double* lb = c.lbuf;  // L block, lower part; column BS holds 1/L[c][c]
  // buf aliases the TMA ring: every compute warp must be done reading its last stage.
  bar_sync(kBarCompute, kComputeThreads);
  {
    const int wm = c.warp >> 2, wn = c.warp & 3;
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
        *reinterpret_cast<double2*>(xb + r * P + cc) = v;
      }
    for (int idx = tid; idx < BS * BS; idx += kComputeThreads) {
      const int r = idx / BS, cc = idx - r * BS;
      if (cc <= r) lb[r * P + cc] = __ldcg(Ld + (int64_t)r * ldl + cc);
    }
    if (tid < BS) lb[tid * P + BS] = 1.0 / __ldcg(Ld + (int64_t)tid * ldl + tid);
  }
  bar_sync(kBarCompute, kComputeThreads);
#pragma unroll 1
  for (int c0 = 0; c0 < BS; c0 += 8) {
    // (a) panel substitution, one thread per row
    if (tid < BS) {
      double v[8];
      double* xr = xb + tid * P + c0;
#pragma unroll
      for (int j = 0; j < 8; j += 2) {
        const double2 q = *reinterpret_cast<const double2*>(xr + j);
        v[j] = q.x;
        v[j + 1] = q.y;
      }
#pragma unroll
      for (int j = 0; j < 8; ++j) {
        v[j] *= lb[(c0 + j) * P + BS];
#pragma unroll
        for (int j2 = j + 1; j2 < 8; ++j2) v[j2] = fma(-v[j], lb[(c0 + j2) * P + c0 + j], v[j2]);
      }
#pragma unroll
      for (int j = 0; j < 8; j += 2) *reinterpret_cast<double2*>(xr + j) = make_double2(v[j], v[j + 1]);
    }
    bar_sync(kBarCompute, kComputeThreads);
    // (b) trailing update X[:, c0+8:] -= X[:, c0:c0+8] L[c0+8:, c0:c0+8]^T
    const int nN = (BS - c0 - 8) / 8;
    if (nN == 0) break;
    for (int blk = c.warp; blk < (BS / 8) * nN; blk += kComputeWarps) {
      const int mb = blk / nN, nk = blk - mb * nN;
      const int r = mb * 8, q = c0 + 8 + nk * 8;
      double2 d = *reinterpret_cast<const double2*>(xb + (r + g) * P + q + 2 * t);
      smem_dmma_sub8<P>(d.x, d.y, xb, r, c0, lb, q, c0, g, t);
      *reinterpret_cast<double2*>(xb + (r + g) * P + q + 2 * t) = d;
    }
    bar_sync(kBarCompute, kComputeThreads);
  }
  // write the solved block back (coalesced rows)
  for (int idx = tid; idx < BS * (BS / 2); idx += kComputeThreads) {
    const int r = idx / (BS / 2), cc = 2 * (idx - r * (BS / 2));
    __stcg(reinterpret_cast<double2*>(X + (int64_t)r * ldx + cc), *reinterpret_cast<const double2*>(xb + r * P + cc));
  }
  bar_sync(kBarCompute, kComputeThreads);
}

// Cholesky of the BS x BS diagonal block A (ld lda), lower, in shared memory
// (POTRF, L196-199), blocked right-looking over 8-column panels:
//   (a) one warp factors the 8x8 diagonal block (column algorithm of SURVEY §8c),
//   (b) the rows below solve against it (one thread per row),
//   (c) the trailing lower triangle is updated with FP64 DMMA.
// A pivot !(d > 0) records info = col0 + c + 1 with atomicMin (LAPACK convention,
// reading R6).  Compute warps only.
template <int BS>
__device__ __forceinline__ void potf2_block(const Ctx<BS>& c, double* A, int lda, int col0, int* info) {
  using C = Cfg<BS>;
  constexpr int P = C::kPitch;
  const int tid = threadIdx.x, lane = c.lane, g = lane >> 2, t = lane & 3;
  double* a = c.buf;
  bar_sync(kBarCompute, kComputeThreads);  // buf aliases the TMA ring
  for (int idx = tid; idx < BS * BS; idx += kComputeThreads) {
    const int r = idx / BS, cc = idx - r * BS;
    if (cc <= r) a[r * P + cc] = __ldcg(A + (int64_t)r * lda + cc);
  }
  bar_sync(kBarCompute, kComputeThreads);
#pragma unroll 1
  for (int c0 = 0; c0 < BS; c0 += 8) {
    // (a) 8x8 diagonal block, warp 0, lane r < 8 owns row c0 + r
    if (c.warp == 0) {
#pragma unroll
      for (int j = 0; j < 8; ++j) {
        const double d = a[(c0 + j) * P + c0 + j];
        const double ljj = sqrt(d);
        if (lane == 0 && !(d > 0.0)) atomicMin(info, col0 + c0 + j + 1);
        __syncwarp();
        if (lane > j && lane < 8) a[(c0 + lane) * P + c0 + j] = a[(c0 + lane) * P + c0 + j] / ljj;
        if (lane == j) {
          a[(c0 + j) * P + c0 + j] = ljj;
          a[(c0 + j) * P + BS] = 1.0 / ljj;
        }
        __syncwarp();
        if (lane > j && lane < 8) {
          const double lrj = a[(c0 + lane) * P + c0 + j];
          for (int q = j + 1; q <= lane; ++q)
            a[(c0 + lane) * P + c0 + q] = fma(-lrj, a[(c0 + q) * P + c0 + j], a[(c0 + lane) * P + c0 + q]);
        }
        __syncwarp();
      }
    }
    bar_sync(kBarCompute, kComputeThreads);
    const int rows = BS - c0 - 8;
    if (rows == 0) break;
    // (b) panel rows below the diagonal block
    if (tid < rows) {
      double v[8];
      double* ar = a + (c0 + 8 + tid) * P + c0;
#pragma unroll
      for (int j = 0; j < 8; ++j) v[j] = ar[j];
#pragma unroll
      for (int j = 0; j < 8; ++j) {
        v[j] *= a[(c0 + j) * P + BS];
#pragma unroll
        for (int j2 = j + 1; j2 < 8; ++j2) v[j2] = fma(-v[j], a[(c0 + j2) * P + c0 + j], v[j2]);
      }
#pragma unroll
      for (int j = 0; j < 8; ++j) ar[j] = v[j];
    }
    bar_sync(kBarCompute, kComputeThreads);
    // (c) trailing lower update: A[r][q] -= L[r, panel] L[q, panel]^T, 8x8 blocks nk <= mb
    const int nr = rows / 8;
    for (int blk = c.warp; blk < nr * (nr + 1) / 2; blk += kComputeWarps) {
      int mb = 0, rem = blk;
      while (rem > mb) {
        rem -= mb + 1;
        ++mb;
      }
      const int r = c0 + 8 + mb * 8, q = c0 + 8 + rem * 8;
      double2 d = *reinterpret_cast<const double2*>(a + (r + g) * P + q + 2 * t);
      smem_dmma_sub8<P>(d.x, d.y, a, r, c0, a, q, c0, g, t);
      *reinterpret_cast<double2*>(a + (r + g) * P + q + 2 * t) = d;
    }
    bar_sync(kBarCompute, kComputeThreads);
  }
  for (int idx = tid; idx < BS * BS; idx += kComputeThreads) {
    const int r = idx / BS, cc = idx - r * BS;
    if (cc <= r) __stcg(A + (int64_t)r * lda + cc, a[r * P + cc]);
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
  const CPrefetch cp{tile_index(i, j), bm * BS, bn * BS};
  gemm_mainloop(c, tile_index(i, k), bm * BS, tile_index(j, k), bn * BS, 0, c.nb, acc, &cp);
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
    solve_block(c, acc, cb > 0, X + cb * BS, c.nb, L + (int64_t)cb * BS * c.nb + cb * BS, c.nb);
    // X[:, cb] (generic stores) is read by TMA in the next block: complete the stores
    // at L2 (gpu-scope fence), then order them before async-proxy accesses.
    __threadfence();
    fence_proxy_async();
    bar_sync(kBarAll, kThreads);
  }
}

// POTRF_k, inner step b (nested tiled Cholesky of the diagonal tile with block BS):
//   potf2 of block (b, b)
template <int BS>
__device__ __forceinline__ void sub_potrf_diag(Ctx<BS>& c, int k, int b, int* info) {
  double* A = c.tile(k, k) + (int64_t)b * BS * c.nb + b * BS;
  potf2_block(c, A, c.nb, k * c.nb + b * BS, info);
}
//   block (r, b), r > b:  X <- X L_bb^{-T}
template <int BS>
__device__ __forceinline__ void sub_potrf_panel(Ctx<BS>& c, int k, int b, int r) {
  double* T = c.tile(k, k);
  Acc<BS> acc;
  solve_block(c, acc, false, T + (int64_t)r * BS * c.nb + b * BS, c.nb, T + (int64_t)b * BS * c.nb + b * BS, c.nb);
}
//   block (r, q), b < q <= r:  A[r, q] -= L[r, b] L[q, b]^T   (K = BS)
template <int BS>
__device__ __forceinline__ void sub_potrf_update(Ctx<BS>& c, int k, int b, int r, int q) {
  Acc<BS> acc;
  const int64_t t = tile_index(k, k);
  const CPrefetch cp{t, r * BS, q * BS};
  gemm_mainloop(c, t, r * BS, t, q * BS, b * BS, (b + 1) * BS, acc, &cp);
  epi_sub_global(c, acc, c.tile(k, k) + (int64_t)r * BS * c.nb + q * BS, c.nb, r == q);
}

}  // namespace chol
