#include <cstdio>
#include <vector>
#include "tile_ops.cuh"
using namespace chol;
__device__ long long g_ph[64];
__device__ long long g_last;
namespace chol {
template <int BS>
__device__ __forceinline__ void solve_block_T(const Ctx<BS>& c, double* X, int ldx, const double* Ld, int ldl) {
  using C = Cfg<BS>;
  constexpr int P = C::kPitch, NB = BS / 8;
  const int tid = threadIdx.x, g = c.lane >> 2, t = c.lane & 3;
  double* lb = c.lbuf();  // L block; column BS holds 1/L[c][c]
  // every warp must be done with lbuf (previous job / previous column block)
  bar_sync(kBarCompute, kComputeThreads);
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[0] += _t - g_last; g_last = _t; }
  load_block<BS>(lb, Ld, ldl);
  if (tid < BS) lb[tid * P + BS] = 1.0 / __ldcg(Ld + (int64_t)tid * ldl + tid);
  bar_sync(kBarCompute, kComputeThreads);
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[1] += _t - g_last; g_last = _t; }
  if (c.warp < BS / 16) {
    RowX<BS> x;
    const int r0 = 16 * c.warp;
#pragma unroll
    for (int mi = 0; mi < 2; ++mi)
#pragma unroll
      for (int cb = 0; cb < NB; ++cb) {
        const double2 v =
            __ldcg(reinterpret_cast<const double2*>(X + (int64_t)(r0 + 8 * mi + g) * ldx + 8 * cb + 2 * t));
        x.v[mi][cb][0] = v.x;
        x.v[mi][cb][1] = v.y;
      }
    const int qbase = c.lane & ~3;
#pragma unroll
    for (int p = 0; p < NB; ++p) {
      const int c0 = 8 * p;
      // (a) substitution inside the panel: column c0+j is held by lane t = j/2, slot j%2
#pragma unroll
      for (int j = 0; j < 8; ++j) {
        const double rd = lb[(c0 + j) * P + BS];
        const double l0 = lb[(c0 + 2 * t) * P + c0 + j], l1 = lb[(c0 + 2 * t + 1) * P + c0 + j];
#pragma unroll
        for (int mi = 0; mi < 2; ++mi) {
          const double xj = __shfl_sync(0xffffffffu, x.v[mi][p][j & 1], qbase | (j >> 1)) * rd;
          if (t == (j >> 1)) x.v[mi][p][j & 1] = xj;
          if (2 * t > j) x.v[mi][p][0] = fma(-xj, l0, x.v[mi][p][0]);
          if (2 * t + 1 > j) x.v[mi][p][1] = fma(-xj, l1, x.v[mi][p][1]);
        }
      }
      // (b) later column blocks: x[:, cb] -= x[:, p] L[cb rows, p cols]^T
#pragma unroll
      for (int cb = 1; cb < NB; ++cb) {  // constant trip count: fully unrolled, x stays in registers
        if (cb <= p) continue;
        const double2 bv = *reinterpret_cast<const double2*>(lb + (8 * cb + g) * P + c0 + 2 * t);
#pragma unroll
        for (int mi = 0; mi < 2; ++mi) {
          dmma884(x.v[mi][cb][0], x.v[mi][cb][1], -x.v[mi][p][0], bv.x);
          dmma884(x.v[mi][cb][0], x.v[mi][cb][1], -x.v[mi][p][1], bv.y);
        }
      }
    }
#pragma unroll
    for (int mi = 0; mi < 2; ++mi)
#pragma unroll
      for (int cb = 0; cb < NB; ++cb)
        __stcg(reinterpret_cast<double2*>(X + (int64_t)(r0 + 8 * mi + g) * ldx + 8 * cb + 2 * t),
               make_double2(x.v[mi][cb][0], x.v[mi][cb][1]));
  }
  bar_sync(kBarCompute, kComputeThreads);  // lbuf free for the next user; X stores issued
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[2] += _t - g_last; g_last = _t; }
}

// Cholesky of the BS x BS diagonal block A (ld lda), lower, in place (POTRF,
// L196-199).  Register-resident like solve_block: for each 8-column panel, the owner
// warps copy it to shared memory, warp 0 factors its 8x8 diagonal block in registers
// (column algorithm of SURVEY §8c, lanes = rows, shuffles), one thread per row
// solves the rows below, and every warp applies the rank-8 update to its lower
// blocks with FP64 DMMA.  A pivot !(d > 0) records info = col0 + c + 1 with
// atomicMin (LAPACK convention, reading R6).  The strictly upper blocks are never
// stored; the upper halves of diagonal 8x8 blocks are scratch (never read).
template <int BS>
__device__ __forceinline__ void potf2_block_T(const Ctx<BS>& c, double* A, int lda, int col0, int* info) {
  constexpr int NB = BS / 8;
  static_assert(NB % 2 == 0 && NB / 2 <= 7, "paired row blocks; warp 7 factors the diagonal blocks");
  const int g = c.lane >> 2, t = c.lane & 3, qbase = c.lane & ~3;
  double* dd = c.lbuf();        // 8 x 8 diagonal block (pitch 8) + 8 reciprocals
  double* rdv = c.lbuf() + 64;
  bar_sync(kBarCompute, kComputeThreads);  // lbuf / pans reuse
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[0] += _t - g_last; g_last = _t; }
  if (c.warp == 7) {
    // factor warp: its own loop, disjoint from the row-block code (register pressure)
#pragma unroll 1
    for (int p = 0; p < NB; ++p) {
      bar_sync(kBarDiag, 64);  // diagonal block p is in dd
      if (c.lane == 0) factor_8x8(dd, rdv, info, col0 + 8 * p);
      bar_sync(kBarCompute, kComputeThreads);  // L_pp published
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[1] += _t - g_last; g_last = _t; }
      bar_sync(kBarCompute, kComputeThreads);  // panel p published
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[2] += _t - g_last; g_last = _t; }
    }
    bar_sync(kBarCompute, kComputeThreads);
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[3] += _t - g_last; g_last = _t; }
    return;
  }
  const bool active = c.warp < NB / 2;
  const int rb0 = c.warp, rb1 = NB - 1 - c.warp;  // the warp's two row blocks
  double x[NB + 1][2];
#define RB(mi) ((mi) == 0 ? rb0 : rb1)
#define SL(mi, cb) ((mi) == 0 ? (cb) : NB - (cb))
  if (active) {
#pragma unroll
    for (int mi = 0; mi < 2; ++mi)
#pragma unroll
      for (int cb = 0; cb < NB; ++cb) {
        if (cb > RB(mi)) continue;  // strictly upper blocks: never needed
        const double2 v =
            __ldcg(reinterpret_cast<const double2*>(A + (int64_t)(8 * RB(mi) + g) * lda + 8 * cb + 2 * t));
        x[SL(mi, cb)][0] = v.x;
        x[SL(mi, cb)][1] = v.y;
      }
    if (c.warp == 0) {  // hand over the first diagonal block (rb0 = 0, slot 0)
      *reinterpret_cast<double2*>(dd + g * 8 + 2 * t) = make_double2(x[0][0], x[0][1]);
      bar_arrive(kBarDiag, 64);
    }
  }
#pragma unroll
  for (int p = 0; p < NB; ++p) {
    constexpr int kHalf = NB / 2;
    const int pm = p < kHalf ? 0 : 1;              // which of its blocks holds row block p
    const int pw = p < kHalf ? p : NB - 1 - p;     // the warp owning row block p
    double* pan = c.pans() + (p & 1) * BS * kPanelPitch;
    bar_sync(kBarCompute, kComputeThreads);  // L_pp and 1/L[j][j] published
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[4] += _t - g_last; g_last = _t; }
    if (active) {
      if (c.warp == pw) {
        const double2 l = *reinterpret_cast<const double2*>(dd + g * 8 + 2 * t);
        x[SL(pm, p)][0] = l.x;
        x[SL(pm, p)][1] = l.y;
      }
      // (2) rows below the diagonal block: L[r, panel] = A[r, panel] L_pp^{-T}
#pragma unroll
      for (int j = 0; j < 8; ++j) {
        const double rd = rdv[j];
        const double l0 = dd[(2 * t) * 8 + j], l1 = dd[(2 * t + 1) * 8 + j];
#pragma unroll
        for (int mi = 0; mi < 2; ++mi) {
          if (RB(mi) <= p) continue;  // warp-uniform
          double* xs = x[SL(mi, p)];
          const double xj = __shfl_sync(0xffffffffu, xs[j & 1], qbase | (j >> 1)) * rd;
          if (t == (j >> 1)) xs[j & 1] = xj;
          if (2 * t > j) xs[0] = fma(-xj, l0, xs[0]);
          if (2 * t + 1 > j) xs[1] = fma(-xj, l1, xs[1]);
        }
      }
#pragma unroll
      for (int mi = 0; mi < 2; ++mi)
        if (RB(mi) > p)
          *reinterpret_cast<double2*>(pan + (8 * RB(mi) + g) * kPanelPitch + 2 * t) =
              make_double2(x[SL(mi, p)][0], x[SL(mi, p)][1]);
    }
    bar_sync(kBarCompute, kComputeThreads);  // panel p published; dd / rdv free
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[5] += _t - g_last; g_last = _t; }
    if (active && p + 1 < NB) {
      // (3) rank-8 update of this warp's lower blocks (rb >= cb > p); block (p+1, p+1)
      // first, handed to the factor warp before the rest
      const int nm = (p + 1) < kHalf ? 0 : 1;
      const int nw = (p + 1) < kHalf ? p + 1 : NB - 2 - p;
      if (c.warp == nw) {
        const double2 bv = *reinterpret_cast<const double2*>(pan + (8 * (p + 1) + g) * kPanelPitch + 2 * t);
        double* xd = x[SL(nm, p + 1)];
        dmma884(xd[0], xd[1], -x[SL(nm, p)][0], bv.x);
        dmma884(xd[0], xd[1], -x[SL(nm, p)][1], bv.y);
        *reinterpret_cast<double2*>(dd + g * 8 + 2 * t) = make_double2(xd[0], xd[1]);
        bar_arrive(kBarDiag, 64);
      }
#pragma unroll
      for (int cb = 1; cb < NB; ++cb) {  // constant trip count: fully unrolled, x stays in registers
        if (cb <= p || cb > rb1) continue;  // warp-uniform (rb1 >= rb0)
        const double2 bv = *reinterpret_cast<const double2*>(pan + (8 * cb + g) * kPanelPitch + 2 * t);
#pragma unroll
        for (int mi = 0; mi < 2; ++mi) {
          if (RB(mi) < cb) continue;
          if (cb == p + 1 && mi == nm && c.warp == nw) continue;  // done above
          dmma884(x[SL(mi, cb)][0], x[SL(mi, cb)][1], -x[SL(mi, p)][0], bv.x);
          dmma884(x[SL(mi, cb)][0], x[SL(mi, cb)][1], -x[SL(mi, p)][1], bv.y);
        }
      }
    }
  }
  if (active) {
    // the whole block is written: L on and below the diagonal, zeros above it (the
    // strictly upper triangle of the factor is zero; written here so a diagonal tile
    // can be copied out as soon as its POTRF completes)
#pragma unroll
    for (int mi = 0; mi < 2; ++mi)
#pragma unroll
      for (int cb = 0; cb < NB; ++cb) {
        double2 v = make_double2(0.0, 0.0);
        if (cb < RB(mi)) {
          v = make_double2(x[SL(mi, cb)][0], x[SL(mi, cb)][1]);
        } else if (cb == RB(mi)) {
          v.x = 2 * t <= g ? x[SL(mi, cb)][0] : 0.0;
          v.y = 2 * t + 1 <= g ? x[SL(mi, cb)][1] : 0.0;
        }
        __stcg(reinterpret_cast<double2*>(A + (int64_t)(8 * RB(mi) + g) * lda + 8 * cb + 2 * t), v);
      }
  }
#undef RB
#undef SL
  bar_sync(kBarCompute, kComputeThreads);
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[6] += _t - g_last; g_last = _t; }
}


}
template <int BS>
__global__ void __launch_bounds__(kThreads, 1) k_bench(double* X, double* L, double* A, int ld, int* info, int which) {
  auto c = make_ctx<BS>(nullptr, nullptr, ld, 1);
  Acc<BS> acc;
  if (threadIdx.x == 0) g_last = clock64();
  __syncthreads();
  (void)acc;
  if (which == 0) solve_block_T(c, X, ld, L, ld); else potf2_block_T(c, A, ld, 0, info);
}
int main() {
  constexpr int BS = 96; const int ld = BS;
  std::vector<double> hX(BS * BS), hL(BS * BS, 0.0), hA(BS * BS);
  for (int i = 0; i < BS; ++i) for (int j = 0; j < BS; ++j) {
      hX[i * BS + j] = 0.001 * ((i * 7 + j * 3) % 11);
      hL[i * BS + j] = (j < i) ? 0.01 * ((i + j) % 5) : (j == i ? 2.0 : 0.0);
      hA[i * BS + j] = (i == j) ? BS : 0.1 / (1 + abs(i - j)); }
  double *X, *L, *A; int* info;
  cudaMalloc(&X, BS * BS * 8); cudaMalloc(&L, BS * BS * 8); cudaMalloc(&A, BS * BS * 8); cudaMalloc(&info, 4);
  cudaMemcpy(X, hX.data(), BS * BS * 8, cudaMemcpyHostToDevice);
  cudaMemcpy(L, hL.data(), BS * BS * 8, cudaMemcpyHostToDevice);
  cudaMemcpy(A, hA.data(), BS * BS * 8, cudaMemcpyHostToDevice);
  const int smem = Cfg<BS>::kSmemBytes;
  cudaFuncSetAttribute(k_bench<BS>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
  for (int which = 0; which < 2; ++which) {
    for (int warm = 0; warm < 2; ++warm) {
      long long z[64] = {0};
      cudaMemcpyToSymbol(g_ph, z, sizeof(z));
      k_bench<BS><<<1, kThreads, smem>>>(X, L, A, ld, info, which);
      cudaDeviceSynchronize();
      long long h[64]; cudaMemcpyFromSymbol(h, g_ph, sizeof(h));
      if (warm) { printf("%s:", which ? "potf2" : "solve"); long long tot=0; for (int i = 0; i < 5; ++i) { printf(" %lld", h[i]); tot+=h[i]; } printf("  total %lld\n", tot); }
    }
  }
  printf("%s\n", cudaGetErrorString(cudaGetLastError()));
}
