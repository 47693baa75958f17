#include <cstdio>
#include <vector>
#include "tile_ops.cuh"
using namespace chol;
__device__ long long g_ph[64];
__device__ long long g_last;
namespace chol {
template <int BS>
__device__ __forceinline__ void solve_block_T(const Ctx<BS>& c, Acc<BS>& acc, bool has_acc, double* X, int ldx,
                                            const double* Ld, int ldl) {
  using C = Cfg<BS>;
  constexpr int P = C::kPitch, NB = BS / 8;
  const int tid = threadIdx.x, g = c.lane >> 2, t = c.lane & 3;
  double* lb = c.lbuf;  // L block; column BS holds 1/L[c][c]
  // every warp must be done with lbuf (previous job / previous column block)
  bar_sync(kBarCompute, kComputeThreads);
  if (threadIdx.x == 0) { long long _t = clock64(); g_ph[0] += _t - g_last; g_last = _t; }
  if (has_acc) {  // X -= acc in the GEMM's fragment layout, through global memory (L2)
    const int wm = c.warp >> 2, wn = c.warp & 3;
#pragma unroll
    for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
      for (int ni = 0; ni < C::NI; ++ni) {
        double2* px = reinterpret_cast<double2*>(X + (int64_t)(wm * C::WM + mi * 8 + g) * ldx + wn * C::WN + ni * 8 +
                                                 2 * t);
        double2 v = __ldcg(px);
        v.x -= acc[mi][ni][0];
        v.y -= acc[mi][ni][1];
        __stcg(px, v);
      }
  }
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
      for (int cb = p + 1; cb < NB; ++cb) {
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
  using C = Cfg<BS>;
  const int tid = threadIdx.x, lane = c.lane, wm = c.warp >> 2, wn = c.warp & 3, g = lane >> 2, t = lane & 3;
  double* pans = c.pans;
  double* rdiag = c.lbuf;  // 1/L[c][c] of the current panel (8 doubles)
  Acc<BS> x;
  frag_load(c, x, A, lda);
  bar_sync(kBarCompute, kComputeThreads);  // buf / lbuf reuse
  if (threadIdx.x == 0) { long long _t = clock64(); g_ph[0] += _t - g_last; g_last = _t; }
#pragma unroll 1
  for (int p = 0; p < BS / 8; ++p) {
    const int c0 = 8 * p;
    double* pan = pans + (p & 1) * BS * kPanelPitch;
    frag_to_panel(c, x, p, pan);
    bar_sync(kBarCompute, kComputeThreads);
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[1] += _t - g_last; g_last = _t; }
    if (tid == 0) {  // 8x8 diagonal block: one thread, all 36 entries in registers
      double v[8][8];
#pragma unroll
      for (int r = 0; r < 8; ++r)
#pragma unroll
        for (int q = 0; q <= r; ++q) v[r][q] = pan[(c0 + r) * kPanelPitch + q];
#pragma unroll
      for (int j = 0; j < 8; ++j) {
        const double d = v[j][j];
        if (!(d > 0.0)) atomicMin(info, col0 + c0 + j + 1);
        // one rsqrt on the column's dependency chain: L[j][j] = d * d^{-1/2}, scale = d^{-1/2}
        // (exact for the perfect squares of the integer family; within an ulp otherwise)
        const double rl = rsqrt(d);
        v[j][j] = d * rl;
        rdiag[j] = rl;
#pragma unroll
        for (int r = j + 1; r < 8; ++r) v[r][j] *= rl;
#pragma unroll
        for (int r = j + 1; r < 8; ++r)
#pragma unroll
          for (int q = j + 1; q <= r; ++q) v[r][q] = fma(-v[r][j], v[q][j], v[r][q]);
      }
#pragma unroll
      for (int r = 0; r < 8; ++r)
#pragma unroll
        for (int q = 0; q <= r; ++q) pan[(c0 + r) * kPanelPitch + q] = v[r][q];
    }
    bar_sync(kBarCompute, kComputeThreads);
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[2] += _t - g_last; g_last = _t; }
    const int r = c0 + 8 + tid;
    if (r < BS) {  // rows below the diagonal block: L[r, panel] = A[r, panel] L_dd^{-T}
      double v[8];
      double* pr = pan + r * kPanelPitch;
#pragma unroll
      for (int j = 0; j < 8; j += 2) {
        const double2 q = *reinterpret_cast<const double2*>(pr + j);
        v[j] = q.x;
        v[j + 1] = q.y;
      }
#pragma unroll
      for (int j = 0; j < 8; ++j) {
        v[j] *= rdiag[j];
#pragma unroll
        for (int j2 = j + 1; j2 < 8; ++j2) v[j2] = fma(-v[j], pan[(c0 + j2) * kPanelPitch + j], v[j2]);
      }
#pragma unroll
      for (int j = 0; j < 8; j += 2) *reinterpret_cast<double2*>(pr + j) = make_double2(v[j], v[j + 1]);
    }
    bar_sync(kBarCompute, kComputeThreads);
    if (threadIdx.x == 0) { long long _t = clock64(); g_ph[3] += _t - g_last; g_last = _t; }
    panel_to_frag(c, x, p, pan);
    // rank-8 update of this warp's lower blocks (rb >= cb > p)
    double a[C::MI][2];
#pragma unroll
    for (int mi = 0; mi < C::MI; ++mi) {
      const double* pr = pan + (wm * C::WM + mi * 8 + g) * kPanelPitch;
      a[mi][0] = -pr[t];
      a[mi][1] = -pr[t + 4];
    }
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      const int cb = wn * C::NI + ni;
      if (cb <= p) continue;
      const double* lr = pan + (cb * 8 + g) * kPanelPitch;
      const double b0 = lr[t], b1 = lr[t + 4];
#pragma unroll
      for (int mi = 0; mi < C::MI; ++mi) {
        if (wm * C::MI + mi < cb) continue;
        dmma884(x[mi][ni][0], x[mi][ni][1], a[mi][0], b0);
        dmma884(x[mi][ni][0], x[mi][ni][1], a[mi][1], b1);
      }
    }
  }
  frag_store(c, x, A, lda, true);
  bar_sync(kBarCompute, kComputeThreads);
  if (threadIdx.x == 0) { long long _t = clock64(); g_ph[4] += _t - g_last; g_last = _t; }
}


}
template <int BS>
__global__ void __launch_bounds__(kThreads, 1) k_bench(double* X, double* L, double* A, int ld, int* info, int which) {
  auto c = make_ctx<BS>(nullptr, nullptr, ld, 1);
  Acc<BS> acc;
  if (threadIdx.x == 0) g_last = clock64();
  __syncthreads();
  if (which == 0) solve_block_T(c, acc, false, X, ld, L, ld); else potf2_block_T(c, A, ld, 0, info);
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
