// Triangular solves with the factor held in a plan's tile store:
// A X = B as L Y = B (forward) then L^T X = Y (backward) -- the use of the Cholesky
// factor (A = L L^T "is used to solve" the SPD system).
//
// B200 form.  The right-hand sides live in a padded device buffer W (n x ldw, row-major,
// ldw = RC * nchunks); the unknowns are cut into SB-row blocks (SB = the plan's block, 96
// at nb = 960) and the right-hand sides into chunks of RC columns (1: register-streamed
// sweeps; 32 / 48 / 64 at SB = 96 on FP64 DMMA -- k_sweep_mma, k_sweep_db; 8 / 32 for the
// SIMT sweeps at SB = 64 / 32; chol_solve picks).  One work item = (block row b, chunk)
// computes
//     forward:  Y_b = inv(L_bb) (B_b - sum_{c<b} L_bc Y_c)
//     backward: X_b = inv(L_bb)^T (Y_b - sum_{c>b} L_cb^T X_c)
// where inv(L_bb) is the inverse of the SB x SB diagonal block, computed once per
// factorization (k_diag_inv): the sequential substitution inside a block becomes a small
// product, so the chain from block to block is one flag hop plus one SB x SB x RC product.  Items are claimed in dependency order with an atomic counter by a persistent
// grid (a CTA only waits on items claimed before its own, so every wait ends); a block's
// result is published with a release flag, consumers acquire it.  Each CTA stages the
// L block it needs in shared memory before waiting for the flag, so the HBM read of L
// (the dominant traffic: the lower triangle once per sweep) overlaps the wavefront.
// Arithmetic: FP64 DMMA (m8n8k4) at SB = 96, FP64 FMA in the SIMT sweeps.
#include <cuda.h>
#include <cuda_runtime.h>
#include <stdint.h>

#include <cstdlib>

#include "dev_common.cuh"
#include "solve.h"
#include "taskid.h"

namespace chol {

constexpr int kSolveThreads = 256;

template <int SB, int RC>
struct SolveCfg {
  static constexpr int P = SB + 2;                   // shared pitch (doubles): rows stay 16-byte aligned
  static constexpr int G = kSolveThreads / RC;       // row groups (thread t: column t % RC, group t / RC)
  static constexpr int RPT = SB / G;                 // rows per thread
  static constexpr int kLBytes = SB * P * 8;
  static constexpr int kSmem = 2 * kLBytes + SB * RC * 8 + 16;  // k_sweep: 2 L buffers + Y block + item
  static_assert(SB % G == 0, "rows per thread");
};
constexpr int kInvPitch = 97;  // k_diag_inv (odd pitch: the column-per-thread walks are conflict-free)

// first element of SB-block (R, C), R >= C, of the factor in the tile store (ld = nb)
__device__ __forceinline__ const double* lblock(const double* tiles, int nb, int sb, int R, int C) {
  const int64_t r = (int64_t)R * sb, c = (int64_t)C * sb;
  const int64_t i = r / nb, j = c / nb;
  return tiles + tile_index(i, j) * (int64_t)nb * nb + (r - i * nb) * nb + (c - j * nb);
}

// acc[i] += sum_k Lop[row_i][k] * Ys[k][col]; Lop = Ls (TRANS = false) or Ls^T (TRANS =
// true: the backward sweep reads L_cb^T and inv(L_bb)^T straight from the untransposed
// block -- every lane of a row group reads the same element, a shared-memory broadcast)
template <int SB, int RC, bool TRANS>
__device__ __forceinline__ void block_fma(const double* Ls, const double* Ys, double (&acc)[SolveCfg<SB, RC>::RPT]) {
  using C = SolveCfg<SB, RC>;
  const int col = threadIdx.x % RC, r0 = (threadIdx.x / RC) * C::RPT;
#pragma unroll 4
  for (int k = 0; k < SB; ++k) {
    const double y = Ys[k * RC + col];
#pragma unroll
    for (int i = 0; i < C::RPT; ++i) acc[i] = fma(TRANS ? Ls[k * C::P + r0 + i] : Ls[(r0 + i) * C::P + k], y, acc[i]);
  }
}

// Per diagonal block b (once per factorization): inv_b = inv(L_bb) -- column j by forward
// substitution of e_j (thread j) in shared memory -- and the two chain matrices
// Mf_b = inv_b L_{b,b-1} (forward) and Mb_b = L_{b+1,b} inv_b (backward), all written
// whole (SB x SB, row-major; zeros above the diagonal of inv_b).  aux = [inv | Mf | Mb],
// each nblocks x SB x SB.
template <int SB>
__global__ void __launch_bounds__(kSolveThreads) k_diag_aux(const double* tiles, int nb, int nblocks, double* aux) {
  extern __shared__ __align__(16) double sm[];
  constexpr int P = kInvPitch;
  double* Ls = sm;
  double* Zs = sm + SB * P;  // Zs[r][j] = inv_b
  double* inv = aux;
  double* Mf = aux + (int64_t)nblocks * SB * SB;
  double* Mb = Mf + (int64_t)nblocks * SB * SB;
  for (int b = blockIdx.x; b < nblocks; b += gridDim.x) {
    __syncthreads();
    const double* G = lblock(tiles, nb, SB, b, b);
    for (int e = threadIdx.x; e < SB * SB; e += kSolveThreads)
      Ls[(e / SB) * P + e % SB] = __ldcg(G + (int64_t)(e / SB) * nb + e % SB);
    __syncthreads();
    const int j = threadIdx.x;
    if (j < SB) {
      for (int r = 0; r < j; ++r) Zs[r * P + j] = 0.0;
      Zs[j * P + j] = 1.0 / Ls[j * P + j];
      for (int r = j + 1; r < SB; ++r) {
        double s = 0.0;
        for (int m = j; m < r; ++m) s = fma(Ls[r * P + m], Zs[m * P + j], s);
        Zs[r * P + j] = -s / Ls[r * P + r];
      }
    }
    __syncthreads();
    double* out = inv + (int64_t)b * SB * SB;
    for (int e = threadIdx.x; e < SB * SB; e += kSolveThreads) out[e] = Zs[(e / SB) * P + (e % SB)];
    // Mf_b = inv_b L_{b,b-1}: Ls <- L_{b,b-1}
    if (b > 0) {
      __syncthreads();
      const double* G1 = lblock(tiles, nb, SB, b, b - 1);
      for (int e = threadIdx.x; e < SB * SB; e += kSolveThreads)
        Ls[(e / SB) * P + e % SB] = __ldcg(G1 + (int64_t)(e / SB) * nb + e % SB);
      __syncthreads();
      double* o = Mf + (int64_t)b * SB * SB;
      for (int e = threadIdx.x; e < SB * SB; e += kSolveThreads) {
        const int r = e / SB, c = e % SB;
        double s = 0.0;
        for (int m = 0; m <= r; ++m) s = fma(Zs[r * P + m], Ls[m * P + c], s);
        o[e] = s;
      }
    }
    // Mb_b = L_{b+1,b} inv_b: Ls <- L_{b+1,b}
    if (b + 1 < nblocks) {
      __syncthreads();
      const double* G2 = lblock(tiles, nb, SB, b + 1, b);
      for (int e = threadIdx.x; e < SB * SB; e += kSolveThreads)
        Ls[(e / SB) * P + e % SB] = __ldcg(G2 + (int64_t)(e / SB) * nb + e % SB);
      __syncthreads();
      double* o = Mb + (int64_t)b * SB * SB;
      for (int e = threadIdx.x; e < SB * SB; e += kSolveThreads) {
        const int r = e / SB, c = e % SB;
        double s = 0.0;
        for (int m = c; m < SB; ++m) s = fma(Ls[r * P + m], Zs[m * P + c], s);
        o[e] = s;
      }
    }
  }
}

__device__ __forceinline__ void cp_async16(void* dst, const void* src) {
  asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(smem_u32(dst)), "l"(src) : "memory");
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void cp_async_wait() { asm volatile("cp.async.wait_group %0;" ::"n"(N) : "memory"); }

// rows x cols (doubles, cols even) block at G (ld) -> dst (pitch), 16-byte cp.async chunks
// spread over the CTA: every chunk of the thread in flight at once
template <int ROWS, int COLS, int PITCH>
__device__ __forceinline__ void stage_async(double* dst, const double* G, int64_t ld) {
  constexpr int CH = COLS / 2;
  for (int e = threadIdx.x; e < ROWS * CH; e += kSolveThreads) {
    const int r = e / CH, c2 = 2 * (e - r * CH);
    cp_async16(dst + r * PITCH + c2, G + (int64_t)r * ld + c2);
  }
}

// One sweep (forward: FWD = true) over work items (block row b, chunk ch of RC columns):
//   forward   Y_b = inv_b (B_b - sum_{c<b-1} L_bc Y_c) - Mf_b Y_{b-1}
//   backward  X_b = inv_b^T (Y_b - sum_{c>b+1} L_cb^T X_c) - Mb_b^T X_{b+1}
// (Mf_b = inv_b L_{b,b-1}, Mb_b = L_{b+1,b} inv_b, k_diag_aux), so only the last product
// waits for the previous block row: the chain from block to block is one flag hop, one
// fetch of the 8- or 32-column block and one SB x SB x RC FMA pass.  Stages: the nc-1
// older off-diagonal blocks (accumulate), the inverse applied to (rhs - acc), then the
// chain matrix against the previous block row.  Each stage's SB x SB matrix streams into
// the other shared buffer (cp.async) while the previous stage computes; the right-hand
// side block sits in registers from the start of the item.  flags[b * nchunks + ch] =
// epoch once block b of chunk ch is final in W.
template <int SB, int RC, bool FWD>
__global__ void __launch_bounds__(kSolveThreads, 1)
    k_sweep(const double* tiles, int nb, int nblocks, const double* aux, double* W, int ldw, int nchunks, int* flags,
            int* counter, int epoch, uint64_t* trace) {
  using C = SolveCfg<SB, RC>;
  extern __shared__ __align__(16) double sm[];
  double* Lb[2] = {sm, sm + SB * C::P};
  double* Ys = sm + 2 * SB * C::P;
  int* s_item = reinterpret_cast<int*>(Ys + SB * RC);
  const int col = threadIdx.x % RC, r0 = (threadIdx.x / RC) * C::RPT;
  const int total = nblocks * nchunks;
  const int64_t bsz = (int64_t)SB * SB;
  const double* inv = aux;
  const double* Mch = aux + (FWD ? 1 : 2) * (int64_t)nblocks * bsz;
  while (true) {
    __syncthreads();
    if (threadIdx.x == 0) *s_item = atomicAdd(counter, 1);
    __syncthreads();
    const int item = *s_item;
    if (item >= total) break;
    uint64_t tr_claim = 0, tr_wait = 0, tr_chain0 = 0, tr_chain1 = 0;
    if (trace && threadIdx.x == 0) tr_claim = globaltimer_ns();
    const int ch = item % nchunks;
    const int b = FWD ? item / nchunks : nblocks - 1 - item / nchunks;
    const int nc = FWD ? b : nblocks - 1 - b;  // block rows this one depends on
    const int nold = nc > 0 ? nc - 1 : 0;      // accumulated before the inverse
    // stage q: q < nold off-diagonal block c(q); q == nold the inverse; q == nold + 1 the chain matrix
    const int nst = nold + 1 + (nc > 0 ? 1 : 0);
    auto cof = [&](int q) { return FWD ? q : nblocks - 1 - q; };  // block row consumed by stage q < nold
    auto stage_L = [&](int q, double* dst) {
      if (q < nold) {
        const int c = cof(q);
        stage_async<SB, SB, C::P>(dst, FWD ? lblock(tiles, nb, SB, b, c) : lblock(tiles, nb, SB, c, b), nb);
      } else if (q == nold) {
        stage_async<SB, SB, C::P>(dst, inv + b * bsz, SB);
      } else {
        stage_async<SB, SB, C::P>(dst, Mch + b * bsz, SB);
      }
      cp_async_commit();
    };
    double* Wb = W + (int64_t)b * SB * ldw + ch * RC;
    double rhs[C::RPT], acc[C::RPT];
#pragma unroll
    for (int i = 0; i < C::RPT; ++i) {
      rhs[i] = __ldcg(Wb + (int64_t)(r0 + i) * ldw + col);
      acc[i] = 0.0;
    }
    stage_L(0, Lb[0]);
    for (int q = 0; q < nst; ++q) {
      const int buf = q & 1;
      if (q != nold) {  // consumes a finished block row: c(q) or the previous row
        const int c = q < nold ? cof(q) : (FWD ? b - 1 : b + 1);
        if (threadIdx.x == 0) {
          const int* f = flags + c * nchunks + ch;
          const uint64_t tw0 = trace ? globaltimer_ns() : 0;
          int v;
          do {
            asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(f) : "memory");
          } while (v != epoch);
          if (trace) {
            const uint64_t tw1 = globaltimer_ns();
            if (q == nold + 1) tr_chain0 = tw0, tr_chain1 = tw1;
            else tr_wait += tw1 - tw0;
          }
        }
        __syncthreads();
        stage_async<SB, RC, RC>(Ys, W + (int64_t)c * SB * ldw + ch * RC, ldw);
        cp_async_commit();
      } else {  // rhs - acc, for the inverse
#pragma unroll
        for (int i = 0; i < C::RPT; ++i) {
          Ys[(r0 + i) * RC + col] = rhs[i] - acc[i];
          acc[i] = 0.0;
        }
        cp_async_commit();  // empty group: keeps the group count uniform
      }
      if (q + 1 < nst) {
        stage_L(q + 1, Lb[buf ^ 1]);  // prefetch the next matrix (its buffer was freed by stage q-1)
        cp_async_wait<1>();           // everything but that prefetch has landed
      } else {
        cp_async_wait<0>();
      }
      __syncthreads();
      if (q == nold + 1) {  // acc = U - M y: negate, accumulate, negate back
#pragma unroll
        for (int i = 0; i < C::RPT; ++i) acc[i] = -acc[i];
        block_fma<SB, RC, !FWD>(Lb[buf], Ys, acc);
#pragma unroll
        for (int i = 0; i < C::RPT; ++i) acc[i] = -acc[i];
      } else {
        block_fma<SB, RC, !FWD>(Lb[buf], Ys, acc);
      }
      __syncthreads();  // Ys and Lb[buf] free
    }
#pragma unroll
    for (int i = 0; i < C::RPT; ++i) __stcg(Wb + (int64_t)(r0 + i) * ldw + col, acc[i]);
    // the CTA barrier orders every thread's stores before thread 0's release (cumulative),
    // so one gpu-scope release publishes the whole block
    __syncthreads();
    if (threadIdx.x == 0) {
      int* f = flags + b * nchunks + ch;
      asm volatile("st.release.gpu.global.b32 [%0], %1;" ::"l"(f), "r"(epoch) : "memory");
      if (trace) {
        uint64_t* t = trace + 6 * (int64_t)(item + (FWD ? 0 : total));
        unsigned smid;
        asm volatile("mov.u32 %0, %%smid;" : "=r"(smid));
        t[0] = tr_claim;
        t[1] = tr_chain0;
        t[2] = tr_chain1;
        t[3] = globaltimer_ns();
        t[4] = tr_wait;
        t[5] = ((uint64_t)b << 32) | smid;
      }
    }
  }
}

// Sentinel of the chain buffers: a signalling NaN (quiet bit clear) -- FP64 arithmetic
// only ever produces quiet NaNs, so no computed block result can look unpublished.
constexpr unsigned long long kChainEmpty = 0x7FF57FF57FF57FF5ull;
// x[i] = sign * p[i * stride] for i < M, once every value is published: all M loads in
// flight at once (one L2 round trip when the block is there), the batch re-read until none
// is the sentinel.
template <int M>
__device__ __forceinline__ void poll_block(double (&x)[M], const double* p, int stride, double sign) {
  unsigned long long v[M];
  bool empty;
  do {
#pragma unroll
    for (int i = 0; i < M; ++i)
      asm volatile("ld.relaxed.gpu.global.b64 %0, [%1];" : "=l"(v[i]) : "l"(p + i * stride) : "memory");
    empty = false;
#pragma unroll
    for (int i = 0; i < M; ++i) empty |= v[i] == kChainEmpty;
  } while (empty);
#pragma unroll
  for (int i = 0; i < M; ++i) x[i] = sign * __longlong_as_double((long long)v[i]);
}
__global__ void k_fill_u64(unsigned long long* p, int64_t n, unsigned long long v) {
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x)
    p[i] = v;
}

// Single right-hand side (nrhs = 1): register-streamed matrix-vector sweeps, same items
// and recurrences as k_sweep; block results are published through a chain buffer whose
// values double as flags (poll_block) -- no flag round trip, no barrier before publishing.  Warp w owns rows [w*RPW, (w+1)*RPW) of every SB x SB
// matrix it streams and lane l the columns l, l+32, ... (KPL = SB/32), so each warp-load
// is 256 contiguous bytes.  A matrix element is used once, so it is loaded straight into
// registers (no shared-memory staging -- staging 73 KB per stage through cp.async or
// per-row bulk copies capped a CTA at ~17 GB/s, tools/solve_trace.py), the next stage's
// matrix while the current one is multiplied; each warp walks the stages on its own
// (its lanes poll the values of the block row consumed, poll_block), so CTA barriers only frame the
// two reductions of an item.
//   FWD, non-transposed: partial p[i] (warp row i) over the lane's columns, reduced
//       across lanes;
//   BWD, transposed (L_cb^T, inv_b^T, Mb_b^T read from the stored blocks): partial p[j]
//       (column l + 32 j) over the warp's rows, reduced across warps.
template <int SB, bool FWD>
__global__ void __launch_bounds__(kSolveThreads, 1)
    k_sweep_vec(const double* tiles, int nb, int nblocks, const double* aux, double* W, double* chain, int* counter,
                uint64_t* trace) {
  constexpr int RPW = SB / 8, KPL = SB / 32, NP = FWD ? RPW : KPL, RP = 33;
  __shared__ double red[FWD ? SB * RP : 8 * SB];
  __shared__ double xs[SB];
  __shared__ int s_item;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31, t = threadIdx.x;
  const int64_t bsz = (int64_t)SB * SB;
  const double* inv = aux;
  const double* Mch = aux + (FWD ? 1 : 2) * (int64_t)nblocks * bsz;
  double R0[RPW][KPL], R1[RPW][KPL], p[NP];
  auto load = [&](double (&R)[RPW][KPL], const double* G, int64_t ld) {
#pragma unroll
    for (int i = 0; i < RPW; ++i)
#pragma unroll
      for (int j = 0; j < KPL; ++j) R[i][j] = __ldcs(G + (int64_t)(warp * RPW + i) * ld + lane + 32 * j);
  };
  // p (+)= sign * Op(R) x with x = block row c (c >= 0: polled from the chain buffer, where
  // each value appears as soon as its producer stores it) or xs (c < 0)
  auto apply = [&](const double (&R)[RPW][KPL], int c, double sign) {
    const double* xv = c >= 0 ? chain + (int64_t)c * SB : xs;
    if (FWD) {
      double x[KPL];
      if (c >= 0) {
        poll_block<KPL>(x, xv + lane, 32, sign);
      } else {
#pragma unroll
        for (int j = 0; j < KPL; ++j) x[j] = sign * xv[lane + 32 * j];
      }
#pragma unroll
      for (int i = 0; i < RPW; ++i)
#pragma unroll
        for (int j = 0; j < KPL; ++j) p[i] = fma(R[i][j], x[j], p[i]);
    } else {
      double x[RPW];
      if (c >= 0) {
        poll_block<RPW>(x, xv + warp * RPW, 1, sign);
      } else {
#pragma unroll
        for (int i = 0; i < RPW; ++i) x[i] = sign * xv[warp * RPW + i];
      }
#pragma unroll
      for (int i = 0; i < RPW; ++i)
#pragma unroll
        for (int j = 0; j < KPL; ++j) p[j] = fma(R[i][j], x[i], p[j]);
    }
  };
  // CTA reduction of the partials: returns the full sum for row/column t (t < SB)
  auto reduce = [&]() -> double {
    if (FWD) {
#pragma unroll
      for (int i = 0; i < RPW; ++i) red[(warp * RPW + i) * RP + lane] = p[i];
    } else {
#pragma unroll
      for (int j = 0; j < KPL; ++j) red[warp * SB + lane + 32 * j] = p[j];
    }
    __syncthreads();
    double s = 0.0;
    if (t < SB) {
      if (FWD) {
        double s2 = 0.0;
#pragma unroll
        for (int l = 0; l < 32; l += 2) {
          s += red[t * RP + l];
          s2 += red[t * RP + l + 1];
        }
        s += s2;
      } else {
#pragma unroll
        for (int w = 0; w < 8; ++w) s += red[w * SB + t];
      }
    }
    return s;
  };
  while (true) {
    __syncthreads();
    if (t == 0) s_item = atomicAdd(counter, 1);
    __syncthreads();
    const int item = s_item;
    if (item >= nblocks) break;
    uint64_t tr_claim = 0, tr_chain0 = 0, tr_chain1 = 0;
    if (trace && t == 0) tr_claim = globaltimer_ns();
    const int b = FWD ? item : nblocks - 1 - item;
    const int nc = FWD ? b : nblocks - 1 - b;
    const int nold = nc > 0 ? nc - 1 : 0;
    const int nst = nold + 1 + (nc > 0 ? 1 : 0);
    auto mat = [&](int q, const double*& G, int64_t& ld) {
      if (q < nold) {
        const int c = FWD ? q : nblocks - 1 - q;
        G = FWD ? lblock(tiles, nb, SB, b, c) : lblock(tiles, nb, SB, c, b);
        ld = nb;
      } else {
        G = (q == nold ? inv : Mch) + b * bsz;
        ld = SB;
      }
    };
    const double rhs = t < SB ? __ldcg(W + (int64_t)b * SB + t) : 0.0;
#pragma unroll
    for (int i = 0; i < NP; ++i) p[i] = 0.0;
    const double* G;
    int64_t ld;
    mat(0, G, ld);
    load(R0, G, ld);
    for (int q = 0; q < nst; q += 2) {
      // stage q in R0 (next into R1), stage q+1 in R1 (next into R0)
#pragma unroll
      for (int h = 0; h < 2; ++h) {
        const int qq = q + h;
        if (qq >= nst) break;
        double (&Rc)[RPW][KPL] = h ? R1 : R0;
        double (&Rn)[RPW][KPL] = h ? R0 : R1;
        if (qq + 1 < nst) {
          mat(qq + 1, G, ld);
          load(Rn, G, ld);
        }
        if (qq < nold) {
          apply(Rc, FWD ? qq : nblocks - 1 - qq, 1.0);
        } else if (qq == nold) {  // xs = rhs - acc, then p = Op(inv_b) xs
          const double s = nold > 0 ? reduce() : 0.0;
          if (t < SB) xs[t] = rhs - s;
          __syncthreads();
#pragma unroll
          for (int i = 0; i < NP; ++i) p[i] = 0.0;
          apply(Rc, -1, 1.0);
        } else {  // chain: p -= Op(M_b) x_{b -+ 1}
          if (trace && t == 0) tr_chain0 = globaltimer_ns();
          apply(Rc, FWD ? b - 1 : b + 1, -1.0);
          if (trace && t == 0) tr_chain1 = globaltimer_ns();
        }
      }
    }
    const double y = reduce();
    if (t < SB) {
      __stcg(W + (int64_t)b * SB + t, y);
      // publish: every value is its own flag (8-byte stores are single-copy atomic, and
      // arithmetic never yields the signalling-NaN sentinel the buffer was filled with)
      asm volatile("st.relaxed.gpu.global.f64 [%0], %1;" ::"l"(chain + (int64_t)b * SB + t), "d"(y) : "memory");
    }
    if (t == 0) {
      if (trace) {
        uint64_t* tt = trace + 6 * (int64_t)(item + (FWD ? 0 : nblocks));
        unsigned smid;
        asm volatile("mov.u32 %0, %%smid;" : "=r"(smid));
        tt[0] = tr_claim;
        tt[1] = tr_chain0;
        tt[2] = tr_chain1;
        tt[3] = globaltimer_ns();
        tt[4] = 0;
        tt[5] = ((uint64_t)b << 32) | smid;
      }
    }
  }
}

template <int SB>
static cudaError_t solve_vec(const SolveArgs& a, cudaStream_t s, int* nlaunch) {
  const int smem_inv = 2 * SB * kInvPitch * 8;
  cudaError_t e;
  if ((e = cudaFuncSetAttribute(k_diag_aux<SB>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_inv))) return e;
  const int nblocks = (int)(a.n / SB);
  if (!a.inv_valid) {
    k_diag_aux<SB><<<std::min(nblocks, a.sms), kSolveThreads, smem_inv, s>>>(a.tiles, a.nb, nblocks, a.inv);
    ++*nlaunch;
  }
  const int grid = std::min(nblocks, a.sms);
  if ((e = cudaMemsetAsync(a.ctl, 0, 2 * sizeof(int), s))) return e;
  k_fill_u64<<<a.sms, 256, 0, s>>>(reinterpret_cast<unsigned long long*>(a.chain), 2 * a.n, kChainEmpty);
  k_sweep_vec<SB, true><<<grid, kSolveThreads, 0, s>>>(a.tiles, a.nb, nblocks, a.inv, a.W, a.chain, a.ctl,
                                                        a.trace);
  k_sweep_vec<SB, false><<<grid, kSolveThreads, 0, s>>>(a.tiles, a.nb, nblocks, a.inv, a.W, a.chain + a.n,
                                                         a.ctl + 1, a.trace);
  *nlaunch += 3;
  return cudaGetLastError();
}

// 32-column chunks on the FP64 tensor path: k_sweep's items, stages, flags and
// recurrences, with each SB x SB x 32 block product on DMMA (m8n8k4) instead of SIMT FMA
// (the SIMT pass re-reads one shared-memory element per FMA and tops out near 7 TF/s).
// Warp w owns the 8 x 8 output blocks (R, C), R = 3 (w % 4) + {0,1,2}, C = 2 (w / 4) +
// {0,1} of the SB = 96 row x 32 column item; thread (g, t) holds elements (8R + g, 8C + 2t,
// +1) -- the accumulator layout of every DMMA.  The matrix is staged with pitch 100 and
// the right-hand-side block with pitch 36, so every fragment load of a half-warp hits 16
// distinct banks (forward: A[g][t] = L[8R+g][k+t]; backward, transposed: L[k+t][8R+g];
// B[t][g] = Y[k+t][8C+g]).
// RC = 64 (round 2, nrhs > 32): twice the columns per item, so each staged 96 x 96 matrix
// feeds twice the DMMA work and the factor is streamed half as often (warp: 3 x 4 blocks,
// pitch 68 keeps the half-warp fragment loads conflict-free: 68 mod 16 = 4 like 36).
template <bool FWD, int RC>
__global__ void __launch_bounds__(kSolveThreads, 1)
    k_sweep_mma(const double* tiles, int nb, int nblocks, const double* aux, double* W, int ldw, int nchunks,
                int* flags, int* counter, int epoch) {
  constexpr int SB = 96, LP = 100, YP = RC + 4, NI = RC / 16;
  static_assert(RC == 32 || RC == 64, "chunk width");
  extern __shared__ __align__(16) double sm[];
  double* Lb[2] = {sm, sm + SB * LP};
  double* Ys = sm + 2 * SB * LP;
  int* s_item = reinterpret_cast<int*>(Ys + SB * YP);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31, g = lane >> 2, t = lane & 3;
  const int R0 = 3 * (warp & 3), C0 = NI * (warp >> 2);
  const int total = nblocks * nchunks;
  const int64_t bsz = (int64_t)SB * SB;
  const double* inv = aux;
  const double* Mch = aux + (FWD ? 1 : 2) * (int64_t)nblocks * bsz;
  // acc (+)= Op(Ls) Ys over k = 0..SB-1
  auto block_mma = [&](const double* Ls, double (&acc)[3][NI][2]) {
#pragma unroll
    for (int k0 = 0; k0 < SB; k0 += 4) {
      double a[3], bv[NI];
#pragma unroll
      for (int mi = 0; mi < 3; ++mi)
        a[mi] = FWD ? Ls[(8 * (R0 + mi) + g) * LP + k0 + t] : Ls[(k0 + t) * LP + 8 * (R0 + mi) + g];
#pragma unroll
      for (int ni = 0; ni < NI; ++ni) bv[ni] = Ys[(k0 + t) * YP + 8 * (C0 + ni) + g];
#pragma unroll
      for (int mi = 0; mi < 3; ++mi)
#pragma unroll
        for (int ni = 0; ni < NI; ++ni) dmma884(acc[mi][ni][0], acc[mi][ni][1], a[mi], bv[ni]);
    }
  };
  while (true) {
    __syncthreads();
    if (threadIdx.x == 0) *s_item = atomicAdd(counter, 1);
    __syncthreads();
    const int item = *s_item;
    if (item >= total) break;
    const int ch = item % nchunks;
    const int b = FWD ? item / nchunks : nblocks - 1 - item / nchunks;
    const int nc = FWD ? b : nblocks - 1 - b;
    const int nold = nc > 0 ? nc - 1 : 0;
    const int nst = nold + 1 + (nc > 0 ? 1 : 0);
    auto cof = [&](int q) { return FWD ? q : nblocks - 1 - q; };
    auto stage_L = [&](int q, double* dst) {
      if (q < nold) {
        const int c = cof(q);
        stage_async<SB, SB, LP>(dst, FWD ? lblock(tiles, nb, SB, b, c) : lblock(tiles, nb, SB, c, b), nb);
      } else if (q == nold) {
        stage_async<SB, SB, LP>(dst, inv + b * bsz, SB);
      } else {
        stage_async<SB, SB, LP>(dst, Mch + b * bsz, SB);
      }
      cp_async_commit();
    };
    double* Wb = W + (int64_t)b * SB * ldw + ch * RC;
    double rhs[3][NI][2], acc[3][NI][2];
#pragma unroll
    for (int mi = 0; mi < 3; ++mi)
#pragma unroll
      for (int ni = 0; ni < NI; ++ni) {
        const double2 v = __ldcg(reinterpret_cast<const double2*>(Wb + (int64_t)(8 * (R0 + mi) + g) * ldw +
                                                                  8 * (C0 + ni) + 2 * t));
        rhs[mi][ni][0] = v.x;
        rhs[mi][ni][1] = v.y;
        acc[mi][ni][0] = acc[mi][ni][1] = 0.0;
      }
    stage_L(0, Lb[0]);
    for (int q = 0; q < nst; ++q) {
      const int buf = q & 1;
      if (q != nold) {
        const int c = q < nold ? cof(q) : (FWD ? b - 1 : b + 1);
        if (threadIdx.x == 0) {
          const int* f = flags + c * nchunks + ch;
          int v;
          do {
            asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(f) : "memory");
          } while (v != epoch);
        }
        __syncthreads();
        stage_async<SB, RC, YP>(Ys, W + (int64_t)c * SB * ldw + ch * RC, ldw);
        cp_async_commit();
      } else {  // Ys = rhs - acc, for the inverse; acc restarts
#pragma unroll
        for (int mi = 0; mi < 3; ++mi)
#pragma unroll
          for (int ni = 0; ni < NI; ++ni) {
            *reinterpret_cast<double2*>(Ys + (8 * (R0 + mi) + g) * YP + 8 * (C0 + ni) + 2 * t) =
                make_double2(rhs[mi][ni][0] - acc[mi][ni][0], rhs[mi][ni][1] - acc[mi][ni][1]);
            acc[mi][ni][0] = acc[mi][ni][1] = 0.0;
          }
        cp_async_commit();
      }
      if (q + 1 < nst) {
        stage_L(q + 1, Lb[buf ^ 1]);
        cp_async_wait<1>();
      } else {
        cp_async_wait<0>();
      }
      __syncthreads();
      if (q == nold + 1) {  // acc = U - M y
        double m[3][NI][2];
#pragma unroll
        for (int mi = 0; mi < 3; ++mi)
#pragma unroll
          for (int ni = 0; ni < NI; ++ni) m[mi][ni][0] = m[mi][ni][1] = 0.0;
        block_mma(Lb[buf], m);
#pragma unroll
        for (int mi = 0; mi < 3; ++mi)
#pragma unroll
          for (int ni = 0; ni < NI; ++ni) {
            acc[mi][ni][0] -= m[mi][ni][0];
            acc[mi][ni][1] -= m[mi][ni][1];
          }
      } else {
        block_mma(Lb[buf], acc);
      }
      __syncthreads();
    }
#pragma unroll
    for (int mi = 0; mi < 3; ++mi)
#pragma unroll
      for (int ni = 0; ni < NI; ++ni)
        __stcg(reinterpret_cast<double2*>(Wb + (int64_t)(8 * (R0 + mi) + g) * ldw + 8 * (C0 + ni) + 2 * t),
               make_double2(acc[mi][ni][0], acc[mi][ni][1]));
    __syncthreads();
    if (threadIdx.x == 0)
      asm volatile("st.release.gpu.global.b32 [%0], %1;" ::"l"(flags + b * nchunks + ch), "r"(epoch) : "memory");
  }
}

// Round 2 (second session): 48-column items with both operands double-buffered.  k_sweep_mma
// fetches each stage's right-hand-side block after the previous stage's product (one exposed
// L2 round trip per 96 x 96 x RC product: 70% of the DMMA pipe, ncu); here the next stage's
// matrix AND right-hand-side block stream in under the current product.  To fit two 96 x 96
// matrices and two 96 x 48 blocks (221 KB) the rows are unpadded and XOR-swizzled -- element
// (r, c) at r * pitch + (c ^ 4 (r & 3)), which keeps every half-warp fragment load
// conflict-free for both sweeps -- and each thread copies a fixed 16-byte column chunk down a
// row stride (no per-chunk index arithmetic).  A right-hand-side block whose producer flag is
// not up when the prefetch is due (the newest rows of the wavefront; the chain stage always)
// is fetched at its own stage as before.  Same DMMA sequence per accumulator as k_sweep_mma.
__device__ __forceinline__ int swz(int r, int c) { return c ^ ((r & 3) << 2); }

// rows x (2 * CH) block at G (ld) -> dst (pitch, swizzled): thread tid < TPR * CH copies
// column chunk tid % CH of rows tid / CH, tid / CH + TPR, ...
template <int ROWS, int CH, int PITCH>
__device__ __forceinline__ void stage_swz(double* dst, const double* G, int64_t ld) {
  constexpr int TPR = kSolveThreads / CH;  // rows per pass
  const int tid = threadIdx.x;
  if (tid >= TPR * CH) return;
  const int c2 = 2 * (tid % CH);
  int r = tid / CH;
  const double* src = G + (int64_t)r * ld + c2;
  for (; r < ROWS; r += TPR, src += TPR * ld) cp_async16(dst + r * PITCH + swz(r, c2), src);
}

template <bool FWD>
__global__ void __launch_bounds__(kSolveThreads, 1)
    k_sweep_db(const double* tiles, int nb, int nblocks, const double* aux, double* W, int ldw, int nchunks,
               int* flags, int* counter, int epoch) {
  constexpr int SB = 96, RC = 48, NI = 3;
  extern __shared__ __align__(16) double sm[];
  auto Lb = [&](int buf) { return sm + buf * SB * SB; };
  auto Yb = [&](int buf) { return sm + 2 * SB * SB + buf * SB * RC; };
  int* s_item = reinterpret_cast<int*>(sm + 2 * SB * SB + 2 * SB * RC);
  int* s_pref = s_item + 1;  // [2] right-hand-side block of the stage with this parity prefetched
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31, g = lane >> 2, t = lane & 3;
  const int R0 = 3 * (warp & 3), C0 = NI * (warp >> 2);
  const int total = nblocks * nchunks;
  const int64_t bsz = (int64_t)SB * SB;
  const double* inv = aux;
  const double* Mch = aux + (FWD ? 1 : 2) * (int64_t)nblocks * bsz;
  auto block_mma = [&](const double* Ls, const double* Ys, double (&acc)[3][NI][2]) {
#pragma unroll  // all 24 k-steps (measured: 0.7-1% faster than unroll 4)
    for (int k0 = 0; k0 < SB; k0 += 4) {
      double a[3], bv[NI];
#pragma unroll
      for (int mi = 0; mi < 3; ++mi) {
        const int r = 8 * (R0 + mi) + g;
        a[mi] = FWD ? Ls[r * SB + ((k0 + t) ^ ((g & 3) << 2))] : Ls[(k0 + t) * SB + (r ^ (t << 2))];
      }
#pragma unroll
      for (int ni = 0; ni < NI; ++ni) bv[ni] = Ys[(k0 + t) * RC + ((8 * (C0 + ni) + g) ^ (t << 2))];
#pragma unroll
      for (int mi = 0; mi < 3; ++mi)
#pragma unroll
        for (int ni = 0; ni < NI; ++ni) dmma884(acc[mi][ni][0], acc[mi][ni][1], a[mi], bv[ni]);
    }
  };
  while (true) {
    __syncthreads();
    if (threadIdx.x == 0) *s_item = atomicAdd(counter, 1);
    __syncthreads();
    const int item = *s_item;
    if (item >= total) break;
    const int ch = item % nchunks;
    const int b = FWD ? item / nchunks : nblocks - 1 - item / nchunks;
    const int nc = FWD ? b : nblocks - 1 - b;
    const int nold = nc > 0 ? nc - 1 : 0;
    const int nst = nold + 1 + (nc > 0 ? 1 : 0);
    auto cof = [&](int q) { return FWD ? q : nblocks - 1 - q; };
    auto ysrc = [&](int q) { return q < nold ? cof(q) : (FWD ? b - 1 : b + 1); };
    auto flag_up = [&](int q) {
      int v;
      asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(flags + ysrc(q) * nchunks + ch) : "memory");
      return v == epoch;
    };
    auto issue_L = [&](int q) {
      if (q < nold) {
        const int c = cof(q);
        stage_swz<SB, SB / 2, SB>(Lb(q & 1), FWD ? lblock(tiles, nb, SB, b, c) : lblock(tiles, nb, SB, c, b), nb);
      } else {
        stage_swz<SB, SB / 2, SB>(Lb(q & 1), (q == nold ? inv : Mch) + b * bsz, SB);
      }
    };
    auto issue_Y = [&](int q) {
      stage_swz<SB, RC / 2, RC>(Yb(q & 1), W + (int64_t)ysrc(q) * SB * ldw + ch * RC, ldw);
    };
    double* Wb = W + (int64_t)b * SB * ldw + ch * RC;
    double rhs[3][NI][2], acc[3][NI][2];
#pragma unroll
    for (int mi = 0; mi < 3; ++mi)
#pragma unroll
      for (int ni = 0; ni < NI; ++ni) {
        const double2 v = __ldcg(reinterpret_cast<const double2*>(Wb + (int64_t)(8 * (R0 + mi) + g) * ldw +
                                                                  8 * (C0 + ni) + 2 * t));
        rhs[mi][ni][0] = v.x;
        rhs[mi][ni][1] = v.y;
        acc[mi][ni][0] = acc[mi][ni][1] = 0.0;
      }
    // stage 0 (its right-hand-side block only if its producer is done) and the decision for stage 1
    if (threadIdx.x == 0) {
      s_pref[0] = 0 < nold && flag_up(0);
      s_pref[1] = 1 < nold && flag_up(1);
    }
    __syncthreads();
    issue_L(0);
    if (s_pref[0]) issue_Y(0);
    cp_async_commit();
    for (int q = 0; q < nst; ++q) {
      const int buf = q & 1;
      if (q != nold && !s_pref[buf]) {  // the right-hand-side block is fetched now
        if (threadIdx.x == 0)
          while (!flag_up(q)) {
          }
        __syncthreads();
        issue_Y(q);
        cp_async_commit();
      }
      if (q + 1 < nst) {  // the next stage streams in under this one (its buffers are free)
        issue_L(q + 1);
        if (s_pref[buf ^ 1]) issue_Y(q + 1);
        cp_async_commit();
        cp_async_wait<1>();
      } else {
        cp_async_wait<0>();
      }
      if (q == nold) {  // Y = rhs - acc for the inverse; acc restarts
#pragma unroll
        for (int mi = 0; mi < 3; ++mi)
#pragma unroll
          for (int ni = 0; ni < NI; ++ni) {
            const int r = 8 * (R0 + mi) + g;
            *reinterpret_cast<double2*>(Yb(buf) + r * RC + swz(r, 8 * (C0 + ni) + 2 * t)) =
                make_double2(rhs[mi][ni][0] - acc[mi][ni][0], rhs[mi][ni][1] - acc[mi][ni][1]);
            acc[mi][ni][0] = acc[mi][ni][1] = 0.0;
          }
      }
      __syncthreads();
      if (q == nold + 1) {  // acc = U - M y
        double m[3][NI][2];
#pragma unroll
        for (int mi = 0; mi < 3; ++mi)
#pragma unroll
          for (int ni = 0; ni < NI; ++ni) m[mi][ni][0] = m[mi][ni][1] = 0.0;
        block_mma(Lb(buf), Yb(buf), m);
#pragma unroll
        for (int mi = 0; mi < 3; ++mi)
#pragma unroll
          for (int ni = 0; ni < NI; ++ni) {
            acc[mi][ni][0] -= m[mi][ni][0];
            acc[mi][ni][1] -= m[mi][ni][1];
          }
      } else {
        block_mma(Lb(buf), Yb(buf), acc);
      }
      // stage q+2 reuses these buffers: prefetch its block only if its producer is done now
      if (threadIdx.x == 0) s_pref[buf] = q + 2 < nold && flag_up(q + 2);
      __syncthreads();
    }
#pragma unroll
    for (int mi = 0; mi < 3; ++mi)
#pragma unroll
      for (int ni = 0; ni < NI; ++ni)
        __stcg(reinterpret_cast<double2*>(Wb + (int64_t)(8 * (R0 + mi) + g) * ldw + 8 * (C0 + ni) + 2 * t),
               make_double2(acc[mi][ni][0], acc[mi][ni][1]));
    __syncthreads();
    if (threadIdx.x == 0)
      asm volatile("st.release.gpu.global.b32 [%0], %1;" ::"l"(flags + b * nchunks + ch), "r"(epoch) : "memory");
  }
}

static cudaError_t solve_db(const SolveArgs& a, cudaStream_t s, int* nlaunch) {
  constexpr int SB = 96;
  const int smem = (2 * SB * SB + 2 * SB * 48) * 8 + 16, smem_inv = 2 * SB * kInvPitch * 8;
  cudaError_t e;
  if ((e = cudaFuncSetAttribute(k_diag_aux<SB>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_inv))) return e;
  if ((e = cudaFuncSetAttribute(k_sweep_db<true>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem))) return e;
  if ((e = cudaFuncSetAttribute(k_sweep_db<false>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem))) return e;
  const int nblocks = (int)(a.n / SB);
  if (!a.inv_valid) {
    k_diag_aux<SB><<<std::min(nblocks, a.sms), kSolveThreads, smem_inv, s>>>(a.tiles, a.nb, nblocks, a.inv);
    ++*nlaunch;
  }
  const int total = nblocks * a.nchunks;
  const int grid = std::min(total, a.sms);
  if ((e = cudaMemsetAsync(a.ctl, 0, (2 + 2 * (size_t)total) * sizeof(int), s))) return e;
  k_sweep_db<true><<<grid, kSolveThreads, smem, s>>>(a.tiles, a.nb, nblocks, a.inv, a.W, a.ldw, a.nchunks, a.ctl + 2,
                                                     a.ctl, 1);
  k_sweep_db<false><<<grid, kSolveThreads, smem, s>>>(a.tiles, a.nb, nblocks, a.inv, a.W, a.ldw, a.nchunks,
                                                      a.ctl + 2 + total, a.ctl + 1, 1);
  *nlaunch += 2;
  return cudaGetLastError();
}

template <int RC>
static cudaError_t solve_mma(const SolveArgs& a, cudaStream_t s, int* nlaunch) {
  constexpr int SB = 96;
  const int smem = (2 * SB * 100 + SB * (RC + 4)) * 8 + 16, smem_inv = 2 * SB * kInvPitch * 8;
  cudaError_t e;
  if ((e = cudaFuncSetAttribute(k_diag_aux<SB>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_inv))) return e;
  if ((e = cudaFuncSetAttribute(k_sweep_mma<true, RC>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem))) return e;
  if ((e = cudaFuncSetAttribute(k_sweep_mma<false, RC>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem))) return e;
  const int nblocks = (int)(a.n / SB);
  if (!a.inv_valid) {
    k_diag_aux<SB><<<std::min(nblocks, a.sms), kSolveThreads, smem_inv, s>>>(a.tiles, a.nb, nblocks, a.inv);
    ++*nlaunch;
  }
  const int total = nblocks * a.nchunks;
  const int grid = std::min(total, a.sms);
  if ((e = cudaMemsetAsync(a.ctl, 0, (2 + 2 * (size_t)total) * sizeof(int), s))) return e;
  k_sweep_mma<true, RC><<<grid, kSolveThreads, smem, s>>>(a.tiles, a.nb, nblocks, a.inv, a.W, a.ldw, a.nchunks,
                                                           a.ctl + 2, a.ctl, 1);
  k_sweep_mma<false, RC><<<grid, kSolveThreads, smem, s>>>(a.tiles, a.nb, nblocks, a.inv, a.W, a.ldw, a.nchunks,
                                                            a.ctl + 2 + total, a.ctl + 1, 1);
  *nlaunch += 2;
  return cudaGetLastError();
}

template <int SB, int RC>
static cudaError_t solve_sb(const SolveArgs& a, cudaStream_t s, int* nlaunch) {
  using C = SolveCfg<SB, RC>;
  const int smem = C::kSmem, smem_inv = 2 * SB * kInvPitch * 8;
  cudaError_t e;
  if ((e = cudaFuncSetAttribute(k_diag_aux<SB>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_inv))) return e;
  if ((e = cudaFuncSetAttribute(k_sweep<SB, RC, true>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem))) return e;
  if ((e = cudaFuncSetAttribute(k_sweep<SB, RC, false>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem))) return e;
  const int nblocks = (int)(a.n / SB);
  if (!a.inv_valid) {
    k_diag_aux<SB><<<std::min(nblocks, a.sms), kSolveThreads, smem_inv, s>>>(a.tiles, a.nb, nblocks, a.inv);
    ++*nlaunch;
  }
  int per_sm = 0;
  if ((e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_sweep<SB, RC, true>, kSolveThreads, smem))) return e;
  const int total = nblocks * a.nchunks;
  const int grid = std::min(total, std::max(1, per_sm) * a.sms);
  if ((e = cudaMemsetAsync(a.ctl, 0, (2 + 2 * (size_t)total) * sizeof(int), s))) return e;
  int* counters = a.ctl;
  int* flags = a.ctl + 2;
  k_sweep<SB, RC, true><<<grid, kSolveThreads, smem, s>>>(a.tiles, a.nb, nblocks, a.inv, a.W, a.ldw, a.nchunks,
                                                          flags, counters, 1, a.trace);
  k_sweep<SB, RC, false><<<grid, kSolveThreads, smem, s>>>(a.tiles, a.nb, nblocks, a.inv, a.W, a.ldw, a.nchunks,
                                                           flags + total, counters + 1, 1, a.trace);
  *nlaunch += 2;
  return cudaGetLastError();
}

cudaError_t solve_run(const SolveArgs& a, cudaStream_t s, int* nlaunch) {
  if (a.rc == 1) {
    switch (a.sb) {
      case 96: return solve_vec<96>(a, s, nlaunch);
      case 64: return solve_vec<64>(a, s, nlaunch);
      case 32: return solve_vec<32>(a, s, nlaunch);
    }
    return cudaErrorInvalidValue;
  }
  // 32-column chunks at SB = 96 on DMMA (CHOL_SOLVE_SIMT=1: the SIMT sweeps; development switch)
  const char* esimt = getenv("CHOL_SOLVE_SIMT");
  if (a.rc == 48 && a.sb == 96) return solve_db(a, s, nlaunch);
  if (a.rc == 64 && a.sb == 96) return solve_mma<64>(a, s, nlaunch);
  if (a.rc == 32 && a.sb == 96 && !(esimt && esimt[0] == '1')) return solve_mma<32>(a, s, nlaunch);
  const bool narrow = a.rc == 8;
  switch (a.sb) {
    case 96: return narrow ? solve_sb<96, 8>(a, s, nlaunch) : solve_sb<96, 32>(a, s, nlaunch);
    case 64: return narrow ? solve_sb<64, 8>(a, s, nlaunch) : solve_sb<64, 32>(a, s, nlaunch);
    case 32: return narrow ? solve_sb<32, 8>(a, s, nlaunch) : solve_sb<32, 32>(a, s, nlaunch);
  }
  return cudaErrorInvalidValue;
}

}  // namespace chol
