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
#include <utility>

#include "dev_common.cuh"
#include "taskid.h"

namespace chol {

constexpr int kComputeWarps = 8;
constexpr int kComputeThreads = kComputeWarps * 32;
constexpr int kThreads = kComputeThreads;
// The K loop runs in stages of BK = 32: per operand two TMA boxes of kBox = 16 doubles
// (128-byte rows, the 128B-swizzle limit) -- half as many stage hand-offs as 16-wide stages
// (tools/microbench/mainloop_bench: 97.4% -> 98.6% of the DMMA bound per 96x96x960 block),
// in a 3-deep ring (the same 4.6 us of TMA lead as 5 stages of 16).
constexpr int kStages = 3;
constexpr int BK = 32;    // doubles per stage
constexpr int kBox = 16;  // doubles per TMA box row (128 bytes)
constexpr int kBarCompute = 1;  // named barrier id: compute warps only
constexpr int kBarAll = 2;      // named barrier id: all warps
constexpr int kBarDiag = 3;     // named barrier id: panel owner warp -> diagonal-factor warp (potf2_block)
constexpr int kBarPivot = 4;    // potf2_block: factored diagonal block published (factor warp -> row warps)
constexpr int kBarPanel = 5;    // potf2_block: solved panel published (row warps only)


template <int BS>
struct Cfg {
  static constexpr int WM = BS / 2, WN = BS / 4;  // warp tile
  static constexpr int MI = WM / 8, NI = WN / 8;  // m8n8 blocks per warp
  static constexpr int kOpBytes = BS * kBox * 8;  // one TMA box: BS rows x 128 B
  static constexpr int kStageBytes = 4 * kOpBytes; // A box 0, A box 1, B box 0, B box 1
  static constexpr int kPipeBytes = kStages * kStageBytes;
  static constexpr int kPitch = BS + 2;            // doubles; keeps double2 alignment
  static constexpr int kBufBytes = BS * kPitch * 8;
  static constexpr int kBarBytes = 320;               // 21 mbarriers (176 B) + job ring descriptors + progress word
  static constexpr int kPreBytes = 1024;           // scheduler warp: successors of the running job (sched.cu)
  static constexpr int kSmemBytes = kPipeBytes + kBufBytes + kBarBytes + kPreBytes + 1024;
  static_assert(2 * BS * 10 + 160 <= BS * kPitch, "potf2 panels fit in lbuf behind dd / rdv");
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
  // Shared-memory regions: fixed offsets from the 1024-aligned dynamic smem base,
  // recomputed on use (the compiler rematerialises them instead of holding ~24
  // registers of pointers live through the register-hungry in-block routines).
  __device__ static char* base() {
    extern __shared__ __align__(1024) char smem_raw[];
    // pointer arithmetic on smem_raw (not an integer round trip) keeps the shared
    // address space visible to the compiler: LDS/STS instead of generic LD/ST
    const uint32_t mis = static_cast<uint32_t>(__cvta_generic_to_shared(smem_raw)) & 1023u;
    return smem_raw + ((1024u - mis) & 1023u);
  }
  __device__ static char* bars() { return base() + Cfg<BS>::kPipeBytes + Cfg<BS>::kBufBytes; }
  __device__ char* pipe() const { return base(); }  // kStages x {A, B} operand buffers
  __device__ double* buf() const { return reinterpret_cast<double*>(base()); }  // solve buffer (aliases pipe)
  __device__ double* lbuf() const { return reinterpret_cast<double*>(base() + Cfg<BS>::kPipeBytes); }  // BS x kPitch
  __device__ double* pans() const {  // potf2: two BS x 8 panels, in lbuf behind two dd (64) / rdv (8) slots
    return reinterpret_cast<double*>(base() + Cfg<BS>::kPipeBytes) + 160;
  }
  __device__ uint64_t* full() const { return reinterpret_cast<uint64_t*>(bars()); }  // kStages
  __device__ uint64_t* empty() const { return full() + kStages; }                     // kStages
  __device__ uint64_t* cbar() const { return empty() + kStages; }  // C-block prefetch (TMA -> lbuf)
  // warp-specialised persistent kernel only (sched.cu):
  __device__ uint64_t* jfull() const { return cbar() + 1; }  // [2] job descriptor ready
  __device__ uint64_t* jdone() const { return jfull() + 2; } // [2] job finished (compute -> scheduler)
  __device__ uint64_t* lfree() const { return jdone() + 2; } // lbuf released (compute -> producer)
  __device__ uint64_t* tstep() const { return lfree() + 1; } // TRSM column block stored (compute -> producer)
  __device__ uint64_t* cready() const { return tstep() + 1; } // C - acc staged in lbuf (compute -> storer)
  __device__ uint64_t* sfree() const { return cready() + 1; } // staged TRSM block read by the store (storer -> producer)
  __device__ uint64_t* rbar() const { return sfree() + 1; }   // [2] RECV bulk-copy buffers (thread 0 only)
  // 2*kStages + 11 = 21 barriers = 168 bytes; then 2 x 3 int4 job descriptors + producer progress word
  __device__ int4* jdesc() const { return reinterpret_cast<int4*>(bars() + 176); }
  // scheduler warp only: the successor list of the running job's node, preloaded while the
  // job runs (sched.cu SuccPre)
  __device__ static char* pre() { return bars() + Cfg<BS>::kBarBytes; }
  uint32_t it;     // stages consumed so far
  uint32_t cphase; // parity of the next cbar completion
  uint32_t rcount; // RECV bulk copies (thread 0): bit h = parity of the next completion of rbar[h]
  int warp, lane;

  const int* slot_map;  // multi-GPU: store slot of tile (i,j) (tile_index order); null = identity
  __device__ int64_t slot(int i, int j) const {
    const int64_t t = tile_index(i, j);
    return slot_map ? (int64_t)__ldg(slot_map + t) : t;
  }
  __device__ double* tile(int i, int j) const { return tiles + slot(i, j) * (int64_t)nb * nb; }
  __device__ bool issuer() const { return threadIdx.x == 0; }
};

template <int BS>
__device__ __forceinline__ Ctx<BS> make_ctx(const CUtensorMap* map, double* tiles, int nb, int N,
                                            const int* slot_map = nullptr) {
  Ctx<BS> c;
  c.map = map;
  c.tiles = tiles;
  c.slot_map = slot_map;
  c.nb = nb;
  c.N = N;
  if (threadIdx.x == 0) *reinterpret_cast<int*>(c.jdesc() + 6) = 0;
  c.it = 0;
  c.cphase = 0;
  c.rcount = 0;
  c.warp = threadIdx.x >> 5;
  c.lane = threadIdx.x & 31;
  if (threadIdx.x == 0) {
    for (int s = 0; s < kStages; ++s) {
      mbar_init(&c.full()[s], 1);
      mbar_init(&c.empty()[s], kComputeWarps);
    }
    mbar_init(c.cbar(), 1);
    // persistent kernel: jdone / lfree complete when the compute warps AND the storer warp
    // (TMA-store epilogue, sched.cu) have arrived
    for (int e = 0; e < 2; ++e) {
      mbar_init(&c.jfull()[e], 1);
      mbar_init(&c.jdone()[e], kComputeWarps + 1);
    }
    mbar_init(c.lfree(), kComputeWarps + 1);
    mbar_init(c.tstep(), 1);  // the storer: TRSM column block written back (sched.cu)
    mbar_init(c.cready(), kComputeWarps);
    mbar_init(c.sfree(), 1);
    mbar_init(&c.rbar()[0], 1);
    mbar_init(&c.rbar()[1], 1);
    fence_mbar_init();
  }
  if (c.issuer() && map) tma_prefetch_desc(map);
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
__device__ __forceinline__ void prefetch_c_issue(Ctx<BS>& c, int64_t tile, int r0, int c0) {
  fence_proxy_async();
  mbar_arrive_expect_tx(c.cbar(), BS * BS * 8);
  char* dst = reinterpret_cast<char*>(c.lbuf());
#pragma unroll 1
  for (int b = 0; b < BS / 16; ++b) tma_load_3d(dst + b * BS * 128, c.map, c.cbar(), c0 + 16 * b, r0, (int)tile);
}

template <int BS>
__device__ __forceinline__ void prefetch_c(Ctx<BS>& c, int64_t tile, int r0, int c0) {
  if (c.issuer()) prefetch_c_issue(c, tile, r0, c0);
}

// Stage q (ring slot q % kStages): A = rows [ra, ra+BS) x columns [ka, ka+BK) of plane ta of
// map ma, B likewise (rb, kb, tb, mb) -- two 16-wide boxes each.  A-less (ma null) stages
// carry only B (the A operand staged in lbuf).
template <int BS>
__device__ __forceinline__ void issue_stage_ab(Ctx<BS>& c, uint32_t q, const CUtensorMap* ma, int64_t ta, int ra, int ka,
                                               const CUtensorMap* mb, int64_t tb, int rb, int kb) {
  using C = Cfg<BS>;
  const uint32_t st = q % kStages, ph = (q / kStages) & 1;
  mbar_wait(&c.empty()[st], ph ^ 1);  // the previous use of this buffer was released by all warps
  mbar_arrive_expect_tx(&c.full()[st], (ma ? 4 : 2) * C::kOpBytes);
  char* sa = c.pipe() + st * C::kStageBytes;
  if (ma) {
    tma_load_3d(sa, ma, &c.full()[st], ka, ra, (int)ta);
    tma_load_3d(sa + C::kOpBytes, ma, &c.full()[st], ka + kBox, ra, (int)ta);
  }
  tma_load_3d(sa + 2 * C::kOpBytes, mb, &c.full()[st], kb, rb, (int)tb);
  tma_load_3d(sa + 3 * C::kOpBytes, mb, &c.full()[st], kb + kBox, rb, (int)tb);
}
template <int BS>
__device__ __forceinline__ void issue_stage(Ctx<BS>& c, uint32_t q, int64_t ta, int ra, int64_t tb, int rb, int kk) {
  issue_stage_ab(c, q, c.map, ta, ra, kk, c.map, tb, rb, kk);
}
// B-only stage (the A operand is staged in lbuf): BS rows x BK of block `blk` of map m
// (the Dinv workspace of the inverse-form TRSM).
template <int BS>
__device__ __forceinline__ void issue_stage_b(Ctx<BS>& c, uint32_t q, const CUtensorMap* m, int blk, int kk) {
  issue_stage_ab<BS>(c, q, nullptr, 0, 0, 0, m, blk, 0, kk);
}

// Consume one TMA stage: wait for it, DMMA it into acc, release it to the producer.
// a_stage >= 0: the A operand is lbuf (boxes 2 a_stage, 2 a_stage + 1) instead of the
// ring stage's A boxes.  Quarter qt of a stage = box qt/2, half qt%2: thread (g, t) reads
// logical 16-byte chunk 2t + h of its row (k = 4t + 2h, +1 within the box); with the 128B
// swizzle (chunk ^= row & 7) the two rows g, g+1 of one 8-lane phase land on chunks of
// opposite parity -> conflict-free LDS.128.
template <int BS>
__device__ __forceinline__ void consume_stage(Ctx<BS>& c, uint32_t q, Acc<BS>& acc, uint32_t rt_zero,
                                              int a_stage = -1) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  const uint32_t st = q % kStages, ph = (q / kStages) & 1;
  mbar_wait(&c.full()[st], ph);
  const uint32_t sbase = smem_u32(c.pipe()) + st * C::kStageBytes;
  uint32_t dep = 0;
#pragma unroll
  for (int qt = 0; qt < 4; ++qt) {
    const int box = qt >> 1, h = qt & 1;
    const uint32_t As = (a_stage >= 0 ? smem_u32(c.lbuf()) + (uint32_t)(2 * a_stage + box) * BS * 128
                                      : sbase + box * C::kOpBytes) + (wm * C::WM + g) * 128;
    const uint32_t Bs = sbase + (2 + box) * C::kOpBytes + (wn * C::WN + g) * 128;
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
  if (c.lane == (int)(dep & rt_zero)) mbar_arrive(&c.empty()[st]);
}

template <int BS>
__device__ __forceinline__ void zero_acc(Acc<BS>& acc) {
#pragma unroll
  for (int mi = 0; mi < Cfg<BS>::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < Cfg<BS>::NI; ++ni) acc[mi][ni][0] = acc[mi][ni][1] = 0.0;
}

// Consumer side only (warp-specialised kernel: a separate producer issues the stages).
// Software-pipelined by quarter stage (16 k each, two per TMA box): the fragments of the
// next quarter are loaded before the DMMAs of the current one, across stage boundaries
// too (the next stage's full barrier is waited for before its first quarter's loads, which
// run under the last quarter's DMMAs) -- the shared-memory latency hides behind ~36 queued
// DMMAs per warp.  Same DMMA sequence per accumulator as consume_stage (bitwise identical).
// The stage is released after its last DMMAs, predicated on every fragment register of the
// stage (XORed right after the DMMAs that consumed it: no extra stall).
// A_LBUF: the A operand of stage s is lbuf boxes 2s, 2s+1 (a block staged there in the TMA
// box layout, e.g. the TRSM's Y = X[:, cb] - acc); the ring stages then carry B only.
template <int BS, bool A_LBUF = false>
__device__ __forceinline__ void gemm_consume(Ctx<BS>& c, int nst, Acc<BS>& acc) {
  using C = Cfg<BS>;
  zero_acc<BS>(acc);
  const uint32_t rt_zero = threadIdx.y;  // 0, unknown to the compiler (see consume_stage)
  if (nst <= 0) return;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  const uint32_t base = smem_u32(c.pipe());
  const uint32_t aoff = (wm * C::WM + g) * 128, boff = 2 * C::kOpBytes + (wn * C::WN + g) * 128;
  const uint32_t chq0 = ((2 * t) ^ g) << 4, chq1 = ((2 * t + 1) ^ g) << 4;  // logical chunks 2t, 2t+1
  double2 a[2][C::MI], b[2][C::NI];
  // fragments of quarter qt of stage s (ring slot st) into register slot r
  auto load = [&](int r, uint32_t st, int s, int qt) {
    const uint32_t box = (uint32_t)(qt >> 1), ch = (qt & 1) ? chq1 : chq0;
    uint32_t abase;
    if constexpr (A_LBUF) abase = smem_u32(c.lbuf()) + (uint32_t)(2 * s) * BS * 128 + box * BS * 128;
    else abase = base + st * C::kStageBytes + box * C::kOpBytes;
    const uint32_t bbase = base + st * C::kStageBytes + box * C::kOpBytes;
#pragma unroll
    for (int mi = 0; mi < C::MI; ++mi) a[r][mi] = lds128(abase + aoff + mi * 8 * 128 + ch);
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) b[r][ni] = lds128(bbase + boff + ni * 8 * 128 + ch);
  };
  uint32_t dep = 0;
  auto mma = [&](int r) {
#pragma unroll
    for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
      for (int ni = 0; ni < C::NI; ++ni) dmma884(acc[mi][ni][0], acc[mi][ni][1], a[r][mi].x, b[r][ni].x);
#pragma unroll
    for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
      for (int ni = 0; ni < C::NI; ++ni) dmma884(acc[mi][ni][0], acc[mi][ni][1], a[r][mi].y, b[r][ni].y);
#pragma unroll
    for (int mi = 0; mi < C::MI; ++mi) dep ^= __double2loint(a[r][mi].x);
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) dep ^= __double2loint(b[r][ni].x);
  };
  uint32_t q = c.it;
  {
    const uint32_t st = q % kStages;
    mbar_wait(&c.full()[st], (q / kStages) & 1);
    load(0, st, 0, 0);
  }
  for (int s = 0; s < nst; ++s, ++q) {
    const uint32_t st = q % kStages;
    load(1, st, s, 1);
    mma(0);
    load(0, st, s, 2);
    mma(1);
    load(1, st, s, 3);
    mma(0);
    if (s + 1 < nst) {  // next stage, first quarter, while this stage's last DMMAs run
      const uint32_t sn = (q + 1) % kStages;
      mbar_wait(&c.full()[sn], ((q + 1) / kStages) & 1);
      load(0, sn, s + 1, 0);
    }
    mma(1);
    // every fragment of this stage has been loaded (dep): hand the buffer back
    __syncwarp();
    if (c.lane == (int)(dep & rt_zero)) mbar_arrive(&c.empty()[st]);
  }
  c.it += nst;
}

// Issue + consume (all-compute CTA, thread 0 issues kStages-1 stages ahead).
template <int BS>
__device__ __forceinline__ void gemm_mainloop(Ctx<BS>& c, int64_t ta, int ra, int64_t tb, int rb, int kbeg,
                                              int kend, Acc<BS>& acc, const CPrefetch* cpre = nullptr) {
  const int nst = (kend - kbeg) / BK;
  if (c.issuer()) {
    fence_proxy_async();  // operands may have been written by generic stores (this or other SMs)
    const int pre = nst < kStages - 1 ? nst : kStages - 1;
    for (int s = 0; s < pre; ++s) issue_stage(c, c.it + s, ta, ra, tb, rb, kbeg + s * BK);
    if (cpre) prefetch_c(c, cpre->tile, cpre->r0, cpre->c0);
  }
  zero_acc<BS>(acc);
  const uint32_t rt_zero = threadIdx.y;
  for (int s = 0; s < nst; ++s) {
    // keep kStages-1 stages in flight: refill the buffer stage s-1 used
    if (c.issuer() && s + kStages - 1 < nst)
      issue_stage(c, c.it + s + kStages - 1, ta, ra, tb, rb, kbeg + (s + kStages - 1) * BK);
    consume_stage(c, c.it + s, acc, rt_zero);
  }
  c.it += nst;
}

// C[0:BS, 0:BS] -= acc for the BS x BS block at Cblk (leading dimension ldc); the old
// C values come from the lbuf prefetch (prefetch_c), results go to global memory.
// lower_only: diagonal block of a diagonal tile -- only r >= c is written (SYRK, L207-208).
template <int BS>
__device__ __forceinline__ void epi_sub_global(Ctx<BS>& c, const Acc<BS>& acc, double* Cblk, int ldc,
                                               bool lower_only) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  mbar_wait(c.cbar(), c.cphase);
  c.cphase ^= 1;
  const uint32_t cs = smem_u32(c.lbuf());
  // all shared loads first (lds128 is volatile: it would otherwise wait behind each store)
  double2 cv[C::MI][C::NI];
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      const int r = wm * C::WM + mi * 8 + g, cc = wn * C::WN + ni * 8 + 2 * t;
      // box cc/16, row r, logical 16-byte chunk (cc%16)/2, 128B swizzle
      cv[mi][ni] = lds128(cs + (cc >> 4) * (BS * 128) + r * 128 + ((((cc & 15) >> 1) ^ (r & 7)) << 4));
    }
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      const int r = wm * C::WM + mi * 8 + g, cc = wn * C::WN + ni * 8 + 2 * t;
      double2 v = cv[mi][ni];
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

// Persistent kernel (sched.cu): C - acc staged IN PLACE in lbuf, the TMA-prefetched C block
// (BS/16 boxes of BS rows x 128 B, 128B-swizzled -- the layout a TMA store of the same boxes
// reads back), for the storer warp's TMA store; the compute warps do not wait for it.
// lower_only: the strictly upper part of the block keeps C, so the stored block leaves
// memory exactly as epi_sub_global's lower-only stores do.  Ends with the cross-proxy
// fence; the caller arrives on cready.
template <int BS>
__device__ __forceinline__ void epi_sub_stage(Ctx<BS>& c, const Acc<BS>& acc, bool lower_only) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  mbar_wait(c.cbar(), c.cphase);
  c.cphase ^= 1;
  const uint32_t cs = smem_u32(c.lbuf());
  double2 cv[C::MI][C::NI];
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      const int r = wm * C::WM + mi * 8 + g, cc = wn * C::WN + ni * 8 + 2 * t;
      cv[mi][ni] = lds128(cs + (cc >> 4) * (BS * 128) + r * 128 + ((((cc & 15) >> 1) ^ (r & 7)) << 4));
    }
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      const int r = wm * C::WM + mi * 8 + g, cc = wn * C::WN + ni * 8 + 2 * t;
      double2 v = cv[mi][ni];
      if (!lower_only || cc <= r) v.x -= acc[mi][ni][0];
      if (!lower_only || cc + 1 <= r) v.y -= acc[mi][ni][1];
      sts128(cs + (cc >> 4) * (BS * 128) + r * 128 + ((((cc & 15) >> 1) ^ (r & 7)) << 4), v);
    }
  fence_proxy_async_shared();  // generic smem writes -> the TMA store (async proxy)
}

// Persistent kernel (sched.cu), K-loop jobs C -= A B^T: -acc staged in lbuf in the TMA box
// layout (BS/16 boxes of BS rows x 128 B, 128B swizzle), which the storer warp adds to C in
// global memory with TMA reduce-add stores (C + (-acc) == C - acc exactly) -- no C block is
// read into the SM at all.  lower_only: the strictly upper part of the block gets -0.0
// (x + -0.0 == x for every x), so the block's upper triangle is left as it is.  Ends with
// the cross-proxy fence; the caller arrives on cready.
template <int BS>
__device__ __forceinline__ void epi_stage_neg(Ctx<BS>& c, const Acc<BS>& acc, bool lower_only) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  const uint32_t cs = smem_u32(c.lbuf());
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      const int r = wm * C::WM + mi * 8 + g, cc = wn * C::WN + ni * 8 + 2 * t;
      double2 v = make_double2(-acc[mi][ni][0], -acc[mi][ni][1]);
      if (lower_only && cc > r) v.x = -0.0;
      if (lower_only && cc + 1 > r) v.y = -0.0;
      sts128(cs + (cc >> 4) * (BS * 128) + r * 128 + ((((cc & 15) >> 1) ^ (r & 7)) << 4), v);
    }
  fence_proxy_async_shared();
}

// lbuf offset (bytes) of element (r, cc), cc even, of a BS x BS block in the TMA box layout
// (box cc/16, row r, logical 16-byte chunk (cc%16)/2, 128B swizzle)
template <int BS>
__device__ __forceinline__ uint32_t lbuf_off(int r, int cc) {
  return (cc >> 4) * (BS * 128) + r * 128 + ((((cc & 15) >> 1) ^ (r & 7)) << 4);
}

// TRSM row slab, inverse form (sched.cu J_TRSM): Y = C - acc with C = X[:, cb] prefetched
// into lbuf, written back in place -- the A operand of the Dinv product that follows
// (gemm_consume<BS, true>); a compute barrier makes every warp's part visible first.
template <int BS>
__device__ __forceinline__ void trsm_stage_y(Ctx<BS>& c, const Acc<BS>& acc) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  mbar_wait(c.cbar(), c.cphase);
  c.cphase ^= 1;
  const uint32_t cs = smem_u32(c.lbuf());
  double2 cv[C::MI][C::NI];
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni)
      cv[mi][ni] = lds128(cs + lbuf_off<BS>(wm * C::WM + mi * 8 + g, wn * C::WN + ni * 8 + 2 * t));
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      double2 v = cv[mi][ni];
      v.x -= acc[mi][ni][0];
      v.y -= acc[mi][ni][1];
      sts128(cs + lbuf_off<BS>(wm * C::WM + mi * 8 + g, wn * C::WN + ni * 8 + 2 * t), v);
    }
  bar_sync(kBarCompute, kComputeThreads);
}

// ... and Z = acc (the solved column block) staged over Y once every warp has read Y,
// for the storer's TMA store (the caller arrives on cready).
template <int BS>
__device__ __forceinline__ void trsm_stage_z(Ctx<BS>& c, const Acc<BS>& acc) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  bar_sync(kBarCompute, kComputeThreads);
  const uint32_t cs = smem_u32(c.lbuf());
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni)
      sts128(cs + lbuf_off<BS>(wm * C::WM + mi * 8 + g, wn * C::WN + ni * 8 + 2 * t),
             make_double2(acc[mi][ni][0], acc[mi][ni][1]));
  fence_proxy_async_shared();
}

// dst[r*P + c] = src[r*ld + c] for a BS x BS block: 16-byte chunks, every load of
// the thread issued before the first shared store (latency paid once).
template <int BS>
__device__ __forceinline__ void load_block(double* dst, const double* src, int64_t ld) {
  constexpr int P = Cfg<BS>::kPitch, CH = BS / 2, NPT = BS * CH / kComputeThreads;
  // loads in flight per thread (register budget)
  constexpr int BATCH = NPT % 6 == 0 ? 6 : (NPT % 4 == 0 ? 4 : (NPT % 2 == 0 ? 2 : 1));
  static_assert((BS * CH) % kComputeThreads == 0 && NPT % BATCH == 0, "block chunks per thread");
#pragma unroll
  for (int i0 = 0; i0 < NPT; i0 += BATCH) {
    double2 v[BATCH];
#pragma unroll
    for (int i = 0; i < BATCH; ++i) {
      const int idx = threadIdx.x + (i0 + i) * kComputeThreads, r = idx / CH, c2 = idx - r * CH;
      v[i] = __ldcg(reinterpret_cast<const double2*>(src + r * ld + 2 * c2));
    }
#pragma unroll
    for (int i = 0; i < BATCH; ++i) {
      const int idx = threadIdx.x + (i0 + i) * kComputeThreads, r = idx / CH, c2 = idx - r * CH;
      *reinterpret_cast<double2*>(dst + r * P + 2 * c2) = v[i];
    }
  }
}

// Panel buffers for the register-resident in-block algorithms: two BS x 8 panels
// (double-buffered) at the end of lbuf's padding-free tail.  lbuf layout:
//   [0, BS*kPitch)  L block (solve_block) -- pitch kPitch, column BS holds 1/L[c][c]
// The panels live in buf (which aliases the TMA ring; the ring is idle here).
constexpr int kPanelPitch = 10;  // doubles per panel row (8 + 2 pad: fewer bank conflicts)

// Load the BS x BS block at G (ld ldg) into x[][][] in the accumulator fragment
// layout (thread owns rows wm*WM + mi*8 + g, cols wn*WN + ni*8 + 2t, +1).
template <int BS>
__device__ __forceinline__ void frag_load(const Ctx<BS>& c, Acc<BS>& x, const double* G, int64_t ldg) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      const double2 v = __ldcg(reinterpret_cast<const double2*>(G + (int64_t)(wm * C::WM + mi * 8 + g) * ldg +
                                                                wn * C::WN + ni * 8 + 2 * t));
      x[mi][ni][0] = v.x;
      x[mi][ni][1] = v.y;
    }
}

template <int BS>
__device__ __forceinline__ void frag_store(const Ctx<BS>& c, const Acc<BS>& x, double* G, int64_t ldg,
                                           bool lower_blocks_only) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni) {
      const int rb = wm * C::MI + mi, cb = wn * C::NI + ni;
      if (lower_blocks_only && cb > rb) continue;
      __stcg(reinterpret_cast<double2*>(G + (int64_t)(rb * 8 + g) * ldg + cb * 8 + 2 * t),
             make_double2(x[mi][ni][0], x[mi][ni][1]));
    }
}

// Owner warps (those holding 8-column block p) copy that column block of x to the panel.
template <int BS>
__device__ __forceinline__ void frag_to_panel(const Ctx<BS>& c, const Acc<BS>& x, int p, double* pan) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  if (wn != p / C::NI) return;
  const int ni = p % C::NI;
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi) {
    const int r = wm * C::WM + mi * 8 + g;
#pragma unroll
    for (int q = 0; q < C::NI; ++q)
      if (q == ni) *reinterpret_cast<double2*>(pan + r * kPanelPitch + 2 * t) = make_double2(x[mi][q][0], x[mi][q][1]);
  }
}
template <int BS>
__device__ __forceinline__ void panel_to_frag(const Ctx<BS>& c, Acc<BS>& x, int p, const double* pan) {
  using C = Cfg<BS>;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  if (wn != p / C::NI) return;
  const int ni = p % C::NI;
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi) {
    const int r = wm * C::WM + mi * 8 + g;
    const double2 v = *reinterpret_cast<const double2*>(pan + r * kPanelPitch + 2 * t);
#pragma unroll
    for (int q = 0; q < C::NI; ++q)
      if (q == ni) {
        x[mi][q][0] = v.x;
        x[mi][q][1] = v.y;
      }
  }
}

// ---- row layout for the in-block solves: warp w < BS/16 owns rows 16w .. 16w+15 and
// all columns; x[mi][cb] = {X[16w+8mi+g][8cb+2t], X[16w+8mi+g][8cb+2t+1]}.  Rows are
// independent in X L^{-T}, so a warp never waits for another, and the pair a thread
// holds is directly the A operand of a DMMA with k-slot t <-> column 8p+2t (+1).
template <int BS>
struct RowX {
  static constexpr int NB = BS / 8;
  double v[2][NB][2];
};

// X -= acc for one BS x BS block X (ld ldx), acc in the GEMM's fragment layout,
// through global memory (L2): the GEMM part of a TRSM column block, applied before its
// in-block solve (solve_block's barriers order these stores before the solve's loads).
template <int BS>
__device__ __forceinline__ void acc_sub_global(const Ctx<BS>& c, const Acc<BS>& acc, double* X, int ldx) {
  using C = Cfg<BS>;
  const int g = c.lane >> 2, t = c.lane & 3;
  const int wm = c.warp >> 2, wn = c.warp & 3;
  // every load of the thread is issued before its first store (the compiler cannot
  // reorder them itself: with a runtime ldx the rows may alias), so the L2 / HBM latency
  // is paid once per block instead of once per fragment
  double2 v[C::MI][C::NI];
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni)
      v[mi][ni] = __ldcg(reinterpret_cast<const double2*>(X + (int64_t)(wm * C::WM + mi * 8 + g) * ldx + wn * C::WN +
                                                          ni * 8 + 2 * t));
#pragma unroll
  for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
    for (int ni = 0; ni < C::NI; ++ni)
      __stcg(reinterpret_cast<double2*>(X + (int64_t)(wm * C::WM + mi * 8 + g) * ldx + wn * C::WN + ni * 8 + 2 * t),
             make_double2(v[mi][ni].x - acc[mi][ni][0], v[mi][ni].y - acc[mi][ni][1]));
}

// Pull rows [0, BS) x columns [c0, c1) of X (ld ldx) towards L2 (prefetch.global.L2,
// fire-and-forget): the not-yet-touched column blocks of a TRSM row slab, whose first
// read (acc_sub_global) would otherwise wait on HBM.
template <int BS>
__device__ __forceinline__ void prefetch_l2_rows(const double* X, int ldx, int c0, int c1) {
  const int lines = (c1 - c0) / 16;  // 128-byte lines per row (c0, c1 multiples of 16)
  for (int e = threadIdx.x; e < BS * lines; e += kComputeThreads) {
    const int r = e / lines, l = e - r * lines;
    asm volatile("prefetch.global.L2 [%0];" ::"l"(X + (int64_t)r * ldx + c0 + 16 * l));
  }
}

// X <- X * Ld^{-T} for one BS x BS block X (ld ldx) against the lower
// triangular BS x BS diagonal block Ld (ld ldl): the in-block part of TRSM
// (L200-202), forward substitution x_c = (b_c - sum_{m<c} x_m L[c][m]) / L[c][c]
// per row, blocked right-looking over 8-column panels: a panel is solved by the four
// lanes of a quad that hold a row (shuffles), then the warp updates its later column
// blocks with FP64 DMMA (X[:, later] -= X[:, panel] L[later, panel]^T).  No CTA
// barrier inside the panel loop.  The block is written back to X.
template <int BS>
__device__ __forceinline__ void solve_block(const Ctx<BS>& c, double* X, int ldx, const double* Ld, int ldl) {
  using C = Cfg<BS>;
  constexpr int P = C::kPitch, NB = BS / 8;
  const int tid = threadIdx.x, g = c.lane >> 2, t = c.lane & 3;
  double* lb = c.lbuf();  // L block; column BS holds 1/L[c][c]
  // every warp must be done with lbuf (previous job / previous column block)
  bar_sync(kBarCompute, kComputeThreads);
  load_block<BS>(lb, Ld, ldl);
  if (tid < BS) lb[tid * P + BS] = 1.0 / __ldcg(Ld + (int64_t)tid * ldl + tid);
  bar_sync(kBarCompute, kComputeThreads);
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
}

// Dinv = L^{-1} for the lower triangular BS x BS block Ld (ld ldl), row-major into Dinv
// (ld BS): the substitution of solve_block applied to the identity, Z L^T = I, so Z =
// L^{-T} and Dinv = Z^T (stored transposed; zeros above the diagonal).  One job per
// diagonal block of L_kk (sched.cu J_INV), off the POTRF chain; the TRSM row slabs then
// apply each diagonal block as a DMMA product with Dinv (reading R19).
template <int BS>
__device__ __forceinline__ void inv_block(const Ctx<BS>& c, const double* Ld, int ldl, double* Dinv) {
  using C = Cfg<BS>;
  constexpr int P = C::kPitch, NB = BS / 8;
  const int tid = threadIdx.x, g = c.lane >> 2, t = c.lane & 3;
  double* lb = c.lbuf();
  bar_sync(kBarCompute, kComputeThreads);
  load_block<BS>(lb, Ld, ldl);
  if (tid < BS) lb[tid * P + BS] = 1.0 / __ldcg(Ld + (int64_t)tid * ldl + tid);
  bar_sync(kBarCompute, kComputeThreads);
  if (c.warp < BS / 16) {
    RowX<BS> x;
    const int r0 = 16 * c.warp;
#pragma unroll
    for (int mi = 0; mi < 2; ++mi)
#pragma unroll
      for (int cb = 0; cb < NB; ++cb) {
        const int r = r0 + 8 * mi + g, cc = 8 * cb + 2 * t;
        x.v[mi][cb][0] = r == cc ? 1.0 : 0.0;
        x.v[mi][cb][1] = r == cc + 1 ? 1.0 : 0.0;
      }
    const int qbase = c.lane & ~3;
#pragma unroll
    for (int p = 0; p < NB; ++p) {
      const int c0 = 8 * p;
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
#pragma unroll
      for (int cb = 1; cb < NB; ++cb) {
        if (cb <= p) continue;
        const double2 bv = *reinterpret_cast<const double2*>(lb + (8 * cb + g) * P + c0 + 2 * t);
#pragma unroll
        for (int mi = 0; mi < 2; ++mi) {
          dmma884(x.v[mi][cb][0], x.v[mi][cb][1], -x.v[mi][p][0], bv.x);
          dmma884(x.v[mi][cb][0], x.v[mi][cb][1], -x.v[mi][p][1], bv.y);
        }
      }
    }
    // Z[r][c] -> Dinv[c][r]
#pragma unroll
    for (int mi = 0; mi < 2; ++mi)
#pragma unroll
      for (int cb = 0; cb < NB; ++cb) {
        const int r = r0 + 8 * mi + g, cc = 8 * cb + 2 * t;
        __stcg(Dinv + (int64_t)cc * BS + r, x.v[mi][cb][0]);
        __stcg(Dinv + (int64_t)(cc + 1) * BS + r, x.v[mi][cb][1]);
      }
  }
  bar_sync(kBarCompute, kComputeThreads);
}
template <int BS>
__device__ __noinline__ void inv_block_job(const double* Ld, int ldl, double* Dinv) {
  Ctx<BS> c{};
  c.warp = threadIdx.x >> 5;
  c.lane = threadIdx.x & 31;
  inv_block(c, Ld, ldl, Dinv);
}

// One thread factors the 8x8 lower block dd (pitch 8) in registers, column by column
// (SURVEY §8c column algorithm), writing L back to dd and 1/L[j][j] to rdv.
__device__ __forceinline__ void factor_8x8(double* dd, double* rdv, int* info, int col) {
  double v[8][8];
#pragma unroll
  for (int r = 0; r < 8; ++r)
#pragma unroll
    for (int q = 0; q <= r; ++q) v[r][q] = dd[r * 8 + q];
#pragma unroll
  for (int j = 0; j < 8; ++j) {
    const double d = v[j][j];
    if (!(d > 0.0)) atomicMin(info, col + j + 1);
    // one rsqrt on the dependency chain: L[j][j] = d * d^{-1/2}, scale = d^{-1/2}
    // (exact for the perfect squares of the integer family; within an ulp otherwise)
    const double rl = rsqrt(d);
    v[j][j] = d * rl;
    rdv[j] = rl;
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
    for (int q = 0; q <= r; ++q) dd[r * 8 + q] = v[r][q];
}

#ifndef POTF2_STAMP
#define POTF2_STAMP(id)  // microbenchmark hook (tools/microbench/potf2_phases.cu)
#endif

// Per-thread state of potf2_block: the warp's two row blocks rb0 = w, rb1 = NB-1-w; slot
// SL(mi, cb) of x holds column block cb of row block mi (cb of the first block in slot
// cb, of the second in slot NB-cb: disjoint since cb <= w < NB-cb).
template <int BS>
struct Potf2Regs {
  static constexpr int NB = BS / 8;
  double x[NB + 1][2];
  int rb0, rb1, g, t, qbase;
  bool active;
  __device__ __forceinline__ int rb(int mi) const { return mi == 0 ? rb0 : rb1; }
  __host__ __device__ static constexpr int sl(int mi, int cb) { return mi == 0 ? cb : NB - cb; }
};

// One 8-column panel P of potf2_block.  P is a template parameter so that every index
// into x is a compile-time constant (a runtime panel index puts x in local memory:
// 208-byte stack frame, 3x slower).  dd / rdv: the slot of panel P (double-buffered by
// parity: the owner of block P+1 hands it over while the other row warps still read L_PP).
template <int BS, int P>
__device__ __forceinline__ void potf2_panel(const Ctx<BS>& c, Potf2Regs<BS>& s, double* dd0) {
  using R = Potf2Regs<BS>;
  constexpr int NB = R::NB, kHalf = NB / 2;
  constexpr int kRowThreads = kHalf * 32;         // row warps 0 .. NB/2-1
  constexpr int pm = P < kHalf ? 0 : 1;           // which of its blocks holds row block P
  constexpr int pw = P < kHalf ? P : NB - 1 - P;  // the warp owning row block P
  double* pan = c.pans() + (P & 1) * BS * kPanelPitch;
  const double* dd = dd0 + (P & 1) * 72;
  const double* rdv = dd + 64;
  const int g = s.g, t = s.t;
  bar_sync(kBarPivot, kRowThreads + 32);  // L_PP and 1/L[j][j] published by the factor warp
  POTF2_STAMP(0);
  if (c.warp == pw) {
    const double2 l = *reinterpret_cast<const double2*>(dd + g * 8 + 2 * t);
    s.x[R::sl(pm, P)][0] = l.x;
    s.x[R::sl(pm, P)][1] = l.y;
  }
  // (2) rows below the diagonal block: L[r, panel] = A[r, panel] L_PP^{-T}
#pragma unroll
  for (int j = 0; j < 8; ++j) {
    const double rd = rdv[j];
    const double l0 = dd[(2 * t) * 8 + j], l1 = dd[(2 * t + 1) * 8 + j];
#pragma unroll
    for (int mi = 0; mi < 2; ++mi) {
      if (s.rb(mi) <= P) continue;  // warp-uniform
      double* xs = s.x[R::sl(mi, P)];
      const double xj = __shfl_sync(0xffffffffu, xs[j & 1], s.qbase | (j >> 1)) * rd;
      if (t == (j >> 1)) xs[j & 1] = xj;
      if (2 * t > j) xs[0] = fma(-xj, l0, xs[0]);
      if (2 * t + 1 > j) xs[1] = fma(-xj, l1, xs[1]);
    }
  }
  if constexpr (P + 1 < NB) {
    // (3a) the owner of row block P+1 updates its diagonal block first -- both operands are
    // its own solved fragments (B[t][g] = L[8(P+1)+g][c0+2t] is the thread's A value) -- and
    // hands it to the factor warp before the panel barrier: the next pivot does not wait
    // for the other row warps' solves
    constexpr int nm = (P + 1) < kHalf ? 0 : 1;
    constexpr int nw = (P + 1) < kHalf ? P + 1 : NB - 2 - P;
    if (c.warp == nw) {
      const double a0 = s.x[R::sl(nm, P)][0], a1 = s.x[R::sl(nm, P)][1];
      double* xd = s.x[R::sl(nm, P + 1)];
      dmma884(xd[0], xd[1], -a0, a0);
      dmma884(xd[0], xd[1], -a1, a1);
      *reinterpret_cast<double2*>(dd0 + ((P + 1) & 1) * 72 + g * 8 + 2 * t) = make_double2(xd[0], xd[1]);
      bar_arrive(kBarDiag, 64);
      POTF2_STAMP(3);
    }
  }
#pragma unroll
  for (int mi = 0; mi < 2; ++mi)
    if (s.rb(mi) > P)
      *reinterpret_cast<double2*>(pan + (8 * s.rb(mi) + g) * kPanelPitch + 2 * t) =
          make_double2(s.x[R::sl(mi, P)][0], s.x[R::sl(mi, P)][1]);
  POTF2_STAMP(1);
  bar_sync(kBarPanel, kRowThreads);  // panel P published
  POTF2_STAMP(2);
  if constexpr (P + 1 < NB) {
    // (3b) rank-8 update of this warp's other lower blocks (rb >= cb > P)
    constexpr int nm = (P + 1) < kHalf ? 0 : 1;
    constexpr int nw = (P + 1) < kHalf ? P + 1 : NB - 2 - P;
#pragma unroll
    for (int cb = P + 1; cb < NB; ++cb) {
      if (cb > s.rb1) continue;  // warp-uniform (rb1 >= rb0)
      const double2 bv = *reinterpret_cast<const double2*>(pan + (8 * cb + g) * kPanelPitch + 2 * t);
#pragma unroll
      for (int mi = 0; mi < 2; ++mi) {
        if (s.rb(mi) < cb) continue;
        if (cb == P + 1 && mi == nm && c.warp == nw) continue;  // done above
        dmma884(s.x[R::sl(mi, cb)][0], s.x[R::sl(mi, cb)][1], -s.x[R::sl(mi, P)][0], bv.x);
        dmma884(s.x[R::sl(mi, cb)][0], s.x[R::sl(mi, cb)][1], -s.x[R::sl(mi, P)][1], bv.y);
      }
    }
    POTF2_STAMP(4);
  }
}

template <int BS, int... P>
__device__ __forceinline__ void potf2_panels(const Ctx<BS>& c, Potf2Regs<BS>& s, double* dd0,
                                             std::integer_sequence<int, P...>) {
  (potf2_panel<BS, P>(c, s, dd0), ...);
}

// Cholesky of the BS x BS diagonal block A (ld lda), lower, in place (POTRF,
// L196-199), blocked right-looking over 8-column panels p, register resident in a
// row layout with paired row blocks: row warp w < NB/2 owns the 8-row blocks rb = w and
// rb = NB-1-w (13 of the 78 lower 8x8 blocks each for BS = 96: balanced work, and
// NB+1 fragment slots per thread instead of 2*NB).  Per panel (potf2_panel):
//   (1) warp 7 factors the diagonal block p with one thread in registers (column
//       algorithm of SURVEY §8c, one rsqrt per column) and publishes it (kBarPivot);
//   (2) every row warp solves its rows below against L_pp (quad shuffles); the owner of
//       row block p+1 at once updates its diagonal block (p+1, p+1) with its own
//       fragments and hands it to warp 7 (kBarDiag) -- the next pivot does not wait for
//       the other row warps' solves or the panel barrier;
//   (3) the row warps publish the panel (kBarPanel, row warps only) and apply the
//       rank-8 update to their other lower blocks with FP64 DMMA.
// The 8x8 diagonal block and its reciprocals are double-buffered by panel parity.
// (Measured and not taken, round 2: the factor warp alone on its SM sub-partition with the
// row warps on warps 0-2 / 4-6, the owner solving its hand-off row block first, and an
// mbarrier instead of kBarPivot -- potf2 alone 39.2K -> 37.0K cycles, but the factorization
// slower: the update DMMAs of six row warps on three sub-partitions.)
// A pivot !(d > 0) records info = col0 + c + 1 with atomicMin (LAPACK convention,
// reading R6).  The block is stored whole: L on and below the diagonal, zeros above.
template <int BS>
__device__ __forceinline__ void potf2_block(const Ctx<BS>& c, double* A, int lda, int col0, int* info) {
  constexpr int NB = BS / 8, kHalf = NB / 2;
  static_assert(NB % 2 == 0 && NB / 2 <= 7, "paired row blocks; warp 7 factors the diagonal blocks");
  using R = Potf2Regs<BS>;
  double* dd0 = c.lbuf();  // two slots of 8 x 8 diagonal block (pitch 8) + 8 reciprocals (72 doubles)
  bar_sync(kBarCompute, kComputeThreads);  // lbuf / pans reuse
  if (c.warp == 7) {
    // factor warp: its own loop, disjoint from the row-block code (register pressure)
#pragma unroll 1
    for (int p = 0; p < NB; ++p) {
      bar_sync(kBarDiag, 64);  // diagonal block p is in its slot
      POTF2_STAMP(5);
      double* dd = dd0 + (p & 1) * 72;
      if (c.lane == 0) factor_8x8(dd, dd + 64, info, col0 + 8 * p);
      POTF2_STAMP(6);
      __syncwarp();
      bar_arrive(kBarPivot, kHalf * 32 + 32);  // L_pp published to the row warps
    }
    bar_sync(kBarCompute, kComputeThreads);
    return;
  }
  if (c.warp >= kHalf) {  // no row blocks
    bar_sync(kBarCompute, kComputeThreads);
    return;
  }
  R s;
  s.g = c.lane >> 2;
  s.t = c.lane & 3;
  s.qbase = c.lane & ~3;
  s.active = true;
  s.rb0 = c.warp;
  s.rb1 = NB - 1 - c.warp;
  const int g = s.g, t = s.t;
#pragma unroll
  for (int mi = 0; mi < 2; ++mi)
#pragma unroll
    for (int cb = 0; cb < NB; ++cb) {
      if (cb > s.rb(mi)) continue;  // strictly upper blocks: never needed
      const double2 v =
          __ldcg(reinterpret_cast<const double2*>(A + (int64_t)(8 * s.rb(mi) + g) * lda + 8 * cb + 2 * t));
      s.x[R::sl(mi, cb)][0] = v.x;
      s.x[R::sl(mi, cb)][1] = v.y;
    }
  if (c.warp == 0) {  // hand over the first diagonal block (rb0 = 0, slot 0)
    *reinterpret_cast<double2*>(dd0 + g * 8 + 2 * t) = make_double2(s.x[0][0], s.x[0][1]);
    bar_arrive(kBarDiag, 64);
  }
  potf2_panels<BS>(c, s, dd0, std::make_integer_sequence<int, NB>{});
  // the whole block is written: L on and below the diagonal, zeros above it (the
  // strictly upper triangle of the factor is zero; written here so a diagonal tile
  // can be copied out as soon as its POTRF completes)
#pragma unroll
  for (int mi = 0; mi < 2; ++mi)
#pragma unroll
    for (int cb = 0; cb < NB; ++cb) {
      double2 v = make_double2(0.0, 0.0);
      if (cb < s.rb(mi)) {
        v = make_double2(s.x[R::sl(mi, cb)][0], s.x[R::sl(mi, cb)][1]);
      } else if (cb == s.rb(mi)) {
        v.x = 2 * t <= g ? s.x[R::sl(mi, cb)][0] : 0.0;
        v.y = 2 * t + 1 <= g ? s.x[R::sl(mi, cb)][1] : 0.0;
      }
      __stcg(reinterpret_cast<double2*>(A + (int64_t)(8 * s.rb(mi) + g) * lda + 8 * cb + 2 * t), v);
    }
  bar_sync(kBarCompute, kComputeThreads);
}

// ------------------------------------------------------------------ sub-tasks
// Each is executed by all warps of one CTA.  Sub-task granularity: a BS x BS
// block (GEMM / SYRK / POTRF-inner), a BS-row slab (TRSM).

// GEMM_i_j_k sub-task (bm, bn):  A_ij[bm, bn] -= L_ik[bm, :] L_jk[bn, :]^T   (L203-206)
// SYRK_j_k  sub-task (bm >= bn): the same with i = j, lower part only      (L207-208)
template <int BS>
__device__ __forceinline__ void sub_update(Ctx<BS>& c, int i, int j, int k, int bm, int bn) {
  Acc<BS> acc;
  const CPrefetch cp{c.slot(i, j), bm * BS, bn * BS};
  gemm_mainloop(c, c.slot(i, k), bm * BS, c.slot(j, k), bn * BS, 0, c.nb, acc, &cp);
  epi_sub_global(c, acc, c.tile(i, j) + (int64_t)bm * BS * c.nb + bn * BS, c.nb, i == j && bm == bn);
}

// TRSM_i_k sub-task = row slab `slab` of A_ik:  X <- X L_kk^{-T}  (L200-202),
// left-looking over BS-column blocks: X[:, cb] = (X[:, cb] - X[:, :cb] L[cb, :cb]^T) L[cb, cb]^{-T}.
template <int BS>
__device__ __forceinline__ void sub_trsm(Ctx<BS>& c, int i, int k, int slab) {
  const int nbb = c.nb / BS;
  double* X = c.tile(i, k) + (int64_t)slab * BS * c.nb;
  const double* L = c.tile(k, k);
  prefetch_l2_rows<BS>(X, c.nb, BS, c.nb);
  for (int cb = 0; cb < nbb; ++cb) {
    Acc<BS> acc;
    if (cb > 0) gemm_mainloop(c, c.slot(i, k), slab * BS, c.slot(k, k), cb * BS, 0, cb * BS, acc);
    if (cb > 0) acc_sub_global(c, acc, X + cb * BS, c.nb);
    solve_block(c, X + cb * BS, c.nb, L + (int64_t)cb * BS * c.nb + cb * BS, c.nb);
    // X[:, cb] (generic stores) is read by TMA in the next block: complete the stores
    // at L2 (gpu-scope fence), then order them before async-proxy accesses.
    __threadfence();
    fence_proxy_async();
    bar_sync(kBarAll, kThreads);
  }
}

// The same row slab in the inverse form of the persistent scheduler's J_TRSM (reading R19):
// per column block cb, Y = X[:, cb] - X[:, :cb] L[cb, :cb]^T staged in lbuf, then
// X[:, cb] = Y Dinv_cb^T with Dinv_cb = inv(L[cb, cb]) (inv_block, computed by k_inv before
// the TRSM batch).  Same DMMA order per accumulator as the scheduler's path, so the factor
// is bitwise identical across executors (R15); here Z is written back with global stores.
template <int BS>
__device__ __forceinline__ void sub_trsm_inv(Ctx<BS>& c, const CUtensorMap* dmap, int i, int k, int slab) {
  using C = Cfg<BS>;
  const int nbb = c.nb / BS;
  const int wm = c.warp >> 2, wn = c.warp & 3, g = c.lane >> 2, t = c.lane & 3;
  double* X = c.tile(i, k) + (int64_t)slab * BS * c.nb;
  prefetch_l2_rows<BS>(X, c.nb, BS, c.nb);
  const uint32_t rt_zero = threadIdx.y;
  for (int cb = 0; cb < nbb; ++cb) {
    {
      Acc<BS> acc;
      if (cb > 0)
        gemm_mainloop(c, c.slot(i, k), slab * BS, c.slot(k, k), cb * BS, 0, cb * BS, acc);
      else
        zero_acc<BS>(acc);
      prefetch_c(c, c.slot(i, k), slab * BS, cb * BS);  // lbuf is free: barrier ending block cb-1
      trsm_stage_y(c, acc);
    }
    Acc<BS> z;
    constexpr int nst = BS / BK;
    if (c.issuer())
      for (int s = 0; s < kStages - 1 && s < nst; ++s) issue_stage_b(c, c.it + s, dmap, k * nbb + cb, s * BK);
    zero_acc<BS>(z);
    for (int s = 0; s < nst; ++s) {
      if (c.issuer() && s + kStages - 1 < nst)
        issue_stage_b(c, c.it + s + kStages - 1, dmap, k * nbb + cb, (s + kStages - 1) * BK);
      consume_stage(c, c.it + s, z, rt_zero, s);
    }
    c.it += nst;
#pragma unroll
    for (int mi = 0; mi < C::MI; ++mi)
#pragma unroll
      for (int ni = 0; ni < C::NI; ++ni)
        __stcg(reinterpret_cast<double2*>(X + (int64_t)(wm * C::WM + mi * 8 + g) * c.nb + cb * BS + wn * C::WN +
                                          ni * 8 + 2 * t),
               make_double2(z[mi][ni][0], z[mi][ni][1]));
    // X[:, cb] is read by TMA in the next block's GEMM; every warp is done with lbuf
    __threadfence();
    fence_proxy_async();
    bar_sync(kBarAll, kThreads);
  }
}

// POTRF_k, inner step b (nested tiled Cholesky of the diagonal tile with block BS):
//   potf2 of block (b, b)
template <int BS>
__device__ __forceinline__ void potf2_job(double* A, int lda, int col0, int* info) {
  // out of line with plain arguments: the in-block factorization gets its own register
  // allocation (it needs ~164 registers) instead of sharing one with the GEMM paths
  Ctx<BS> c{};
  c.warp = threadIdx.x >> 5;
  c.lane = threadIdx.x & 31;
  potf2_block(c, A, lda, col0, info);
}
// solve_block out of line with plain arguments, for the persistent kernel (three call
// sites: TRSM slab, TS, POTRF panel): one copy with its own register allocation, so its
// ~100 live registers do not raise the pressure of the GEMM paths around the call sites.
template <int BS>
__device__ __noinline__ void solve_block_job(double* X, int ldx, const double* Ld, int ldl) {
  Ctx<BS> c{};
  c.warp = threadIdx.x >> 5;
  c.lane = threadIdx.x & 31;
  solve_block(c, X, ldx, Ld, ldl);
}
template <int BS>
__device__ __forceinline__ void sub_potrf_diag(Ctx<BS>& c, int k, int b, int* info) {
  double* A = c.tile(k, k) + (int64_t)b * BS * c.nb + b * BS;
  potf2_job<BS>(A, c.nb, k * c.nb + b * BS, info);
}
//   block (r, b), r > b:  X <- X L_bb^{-T}
template <int BS>
__device__ __forceinline__ void sub_potrf_panel(Ctx<BS>& c, int k, int b, int r) {
  double* T = c.tile(k, k);
  solve_block_job<BS>(T + (int64_t)r * BS * c.nb + b * BS, c.nb, T + (int64_t)b * BS * c.nb + b * BS, c.nb);
  // the mirror block (b, r) lies in the strictly upper triangle of L_kk: final as zero
  // (no task reads it; zeroing it here lets the tile be copied out as soon as it is final)
  double* U = T + (int64_t)b * BS * c.nb + r * BS;
  for (int e = threadIdx.x; e < BS * BS / 2; e += kComputeThreads) {
    const int row = e / (BS / 2), col = 2 * (e % (BS / 2));
    __stcg(reinterpret_cast<double2*>(U + (int64_t)row * c.nb + col), make_double2(0.0, 0.0));
  }
}
//   block (r, q), b < q <= r:  A[r, q] -= L[r, b] L[q, b]^T   (K = BS)
template <int BS>
__device__ __forceinline__ void sub_potrf_update(Ctx<BS>& c, int k, int b, int r, int q) {
  Acc<BS> acc;
  const int64_t t = c.slot(k, k);
  const CPrefetch cp{t, r * BS, q * BS};
  gemm_mainloop(c, t, r * BS, t, q * BS, b * BS, (b + 1) * BS, acc, &cp);
  epi_sub_global(c, acc, c.tile(k, k) + (int64_t)r * BS * c.nb + q * BS, c.nb, r == q);
}

}  // namespace chol
