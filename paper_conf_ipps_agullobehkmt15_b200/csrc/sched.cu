// Device-side dependency-counting task scheduler (CHOL_EXEC_SCHEDULER).
//
// PAPER.md §II-B2 / §V-A (L283-306, L633-660): tasks of the Algorithm 1 DAG run as
// soon as their direct data dependencies (L213-220) are satisfied; the policy decides
// which ready task a free worker takes.  B200 form: ONE persistent kernel, one CTA
// per SM ("worker").  Each task is a node with a dependency counter; when it becomes
// ready all its CTA sub-tasks ("jobs") are appended to a device ready queue; a worker
// pops a job, runs the tile op (tile_ops.cuh), and the worker that finishes a node's
// last job decrements the successors' counters and enqueues those reaching zero.
// POTRF_k is a chain of inner nodes (nested tiled Cholesky of the diagonal tile with
// block BS: DIAG b -> PANEL b -> UPDATE b -> DIAG b+1 ...).
//
// Policies (include/chol.h): DYNAMIC = one FIFO; CP_PRIORITY = kBuckets FIFOs keyed by
// the bottom-level of the task (HEFT/dmdas, L299-301, L655-660), a worker takes the
// highest non-empty bucket; STATIC = CP_PRIORITY + POTRF and the TRSMs within
// trsm_pin_distance of the diagonal are pinned to `latency_workers` dedicated CTAs
// (the paper's TRSM-distance rule, L1019-1025).
#include <algorithm>
#include <climits>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <vector>

#include "dag.h"
#include "sched.h"
#include "taskid.h"
#include "tile_ops.cuh"

namespace chol {

constexpr int kBuckets = 64;           // priority buckets per queue class
constexpr int kQueues = 2 * kBuckets;  // [0, 64) normal, [64, 128) pinned
constexpr int kQStride = 32;           // ints between queue heads (separate 128B lines)

// Job types: J_UPD GEMM/SYRK block (K = nb); J_TRSM row slab (left-looking, inverse form:
// per column block one GEMM over the solved blocks and one product with Dinv); J_INV
// Dinv_b = inv(L_kk[b, b]) for the slabs (one per diagonal block of L_kk); (older text:
// default plan); POTRF inner: J_DIAG potf2 of block (b,b), J_PANEL solve of block (r,b),
// J_PUPD K=BS update of block (r,q); TRSM right-looking: J_TS solve of block (s,c) of
// A_ik against L_kk[c,c], J_TU K=BS update A_ik[s,c'] -= A_ik[s,c] L_kk[c',c]^T.
// Multi-GPU: J_RECV copies row slab a of remote panel tile (i, j) from its owner b (peer
// memory over NVLink) into this rank's cache slot.
enum JobType : int16_t {
  J_UPD = 0, J_TRSM = 1, J_DIAG = 2, J_PANEL = 3, J_PUPD = 4, J_TS = 5, J_TU = 6, J_RECV = 7, J_INV = 8,
  J_NOP = 9  // no work: a node that only publishes (host-class TRSM "inputs ready", hetero.cpp)
};
struct Job {
  int16_t type, i, j, k, a, b, c, pad;
};

struct DevSched {
  const Job* jobs;
  const int* job_node;
  int* node_deps;   // remaining predecessors
  int* node_left;   // remaining jobs
  const int* node_job_begin;
  const int* node_job_count;
  const int* succ_off;
  const int* succ;
  const int* node_paper;   // paper-level task id (taskid.h) for the trace
  const int* node_queue;   // queue index
  int* q_items;            // node id + 1 (0 = not yet written)
  int* node_next;          // next job index to hand out within a node
  const int* q_base;       // start of each queue in q_items
  int* q_head;             // kQueues * kQStride
  int* q_tail;             // kQueues * kQStride
  int* done_nodes;
  int* finished;
  const int* abort_flag;   // device word set by the host watchdog (api.cu) to stop a stalled run
  uint64_t* job_trace;     // trace == 2: per job {t0, t1, worker << 32 | smid, t_enqueue}
  const uint64_t* tr_base; // globaltimer at factorization start (trace only)
  int total_nodes;
  int latency_workers;     // STATIC: CTAs [0, latency_workers) serve the pinned queues only
  int policy;
  // ---- multi-GPU (null / 0 on one GPU)
  const int* slot_map;        // local slot of each tile
  const int* owner_slot;      // slot of each tile in its owner's store
  double* const* peer_slots;  // [nranks] slot stores (IPC-mapped; own entry = local)
  int* const* peer_flags;     // [nranks] per-tile "final at epoch" flags of each rank
  int* my_flags;              // this rank's flags (== peer_flags[rank])
  const int* node_publish;    // tile made final by the node (published to the other ranks), -1
  const int4* watch;          // RECV nodes to fire: {node, owner rank, tile, 0}, sorted by step
  int* watch_fired;           // per watch entry
  int nwatch;
  unsigned epoch;             // factorization number (flags hold the epoch they became final in)
  int nb;
  double* dinv;               // [N][nb/BS] BS x BS inverses of the diagonal blocks of each L_kk (J_INV)
};

// ------------------------------------------------------------------ device queue ops
// -DCHOL_HOPS: the scheduler warp of every CTA accumulates clock64 sections of the hand-off
// path (a worker whose completion readies a single-job successor runs it next): [0] jdone
// seen -> node counter decremented, [1] -> successors decremented / taker chosen, [2] ->
// other successors pushed, [3] -> node counted / trace, [4] -> descriptor written (jfull),
// [5] hand-off count, [6] compute end (globaltimer) -> jdone seen (ns).
#ifdef CHOL_HOPS
__device__ unsigned long long g_hop[8];
__device__ long long g_hopt[1024][4];  // per CTA: stamps inside node_done_warp
#define HOP_T(v) const long long v = clock64()
#define HOP_MARK(i) \
  if (lane == 0) g_hopt[blockIdx.x][i] = clock64()
#define HOP_ADD(i, v) \
  if (lane == 0) atomicAdd(&g_hop[i], (unsigned long long)(v))
#else
#define HOP_T(v)
#define HOP_MARK(i)
#define HOP_ADD(i, v)
#endif
__device__ __forceinline__ int ld_volatile(const int* p) { return *reinterpret_cast<const volatile int*>(p); }

// A ready node is enqueued ONCE (one queue item per node); workers then claim its jobs
// one by one with an atomicAdd on the node's job counter (never fails while jobs
// remain -- a CAS-per-job queue serialised dispatch at one job per L2 round trip).
__device__ __forceinline__ void push_node(const DevSched& d, int node) {
  const int q = d.node_queue[node];
  if (d.job_trace) {
    const uint64_t tq = globaltimer_ns() - *d.tr_base;
    const int cnt = d.node_job_count[node], jb = d.node_job_begin[node];
    for (int c = 0; c < cnt; ++c) d.job_trace[4 * (size_t)(jb + c) + 3] = tq;
  }
  const int slot = atomicAdd(&d.q_tail[q * kQStride], 1);
  __threadfence();  // node counters / inputs before the item that publishes the node
  atomicExch(&d.q_items[d.q_base[q] + slot], node + 1);
}

// A node is done (its last job completed, or it has no jobs): publish the tile it makes
// final (multi-GPU / streamed output), release its successors, count it.  Called by a
// whole warp: lane l releases successors l, l+32, ... concurrently (a POTRF diagonal
// block or a TRSM exit node has up to ~2N successors; one push costs two dependent L2
// round trips).  A successor without jobs (the entry / exit node of a block-decomposed
// TRSM) is done as soon as it is ready, by the whole warp; Depth bounds that recursion
// (the builder never chains two job-less nodes).
// Direct handoff: if the calling worker will be idle (can_take), the first ready
// single-job successor is not queued but returned, and the worker runs it next -- no
// queue round trips on chains of single-job nodes (the POTRF block DAG's critical path
// D(b) -> P(b+1,b) -> U(b+1,b+1,b) -> D(b+1)).  Returns that node or -1 (warp-uniform).
template <int Depth>
__device__ int node_done_warp(const DevSched& d, int node, int lane, bool can_take);

// Release the successors succ[beg, end) of a completed node, one lane per edge (see
// node_done_warp); returns the hand-off node or -1 (warp-uniform).
template <int Depth>
__device__ int release_range(const DevSched& d, int beg, int end, int lane, bool can_take) {
  int take = -1;
  for (int e0 = beg; e0 < end; e0 += 32) {
    const int e = e0 + lane;
    int s = -1, cnt = -1;
    if (e < end) {
      s = d.succ[e];
      if (atomicSub(&d.node_deps[s], 1) == 1) cnt = d.node_job_count[s];
    }
    const bool join = Depth > 0 && cnt == 0;
    const unsigned ms = __ballot_sync(0xffffffffu, can_take && take < 0 && cnt == 1);
    const int taker = ms ? __ffs(ms) - 1 : -1;
    if (taker >= 0) {
      HOP_MARK(0);
      take = __shfl_sync(0xffffffffu, s, taker);
      if (lane == taker && d.job_trace) d.job_trace[4 * (size_t)d.node_job_begin[s] + 3] = globaltimer_ns() - *d.tr_base;
    }
    if (cnt > 0 && lane != taker) push_node(d, s);
    if (taker >= 0) {
      __syncwarp();
      HOP_MARK(1);
    }
    if constexpr (Depth > 0) {
      unsigned m = __ballot_sync(0xffffffffu, join);
      while (m) {
        const int src = __ffs(m) - 1;
        m &= m - 1;
        const int t = node_done_warp<Depth - 1>(d, __shfl_sync(0xffffffffu, s, src), lane, can_take && take < 0);
        if (take < 0) take = t;
      }
    }
  }
  return take;
}

// The node's tile is final: release it to every rank (system scope, NVLink) / the host.
__device__ __forceinline__ void publish_node(const DevSched& d, int node, int lane) {
  if (lane == 0 && d.node_publish) {
    const int pt = d.node_publish[node];
    if (pt >= 0) {
      __threadfence_system();
      asm volatile("st.release.sys.global.u32 [%0], %1;" ::"l"(d.my_flags + pt), "r"(d.epoch) : "memory");
    }
  }
}

__device__ __forceinline__ void count_node_done(const DevSched& d, int lane) {
  if (lane == 0 && atomicAdd(d.done_nodes, 1) == d.total_nodes - 1) {
    __threadfence();
    atomicExch(d.finished, 1);
  }
  __syncwarp();
}

template <int Depth>
__device__ int node_done_warp(const DevSched& d, int node, int lane, bool can_take) {
  __threadfence();
  publish_node(d, node, lane);
  const int take = release_range<Depth>(d, d.succ_off[node], d.succ_off[node + 1], lane, can_take);
  count_node_done(d, lane);
  HOP_MARK(2);
  return take;
}

// A node whose dependencies are all satisfied, single thread (init, watcher lanes):
// queue its jobs, or -- job-less -- release its successors at once.
__device__ void ready_node(const DevSched& d, int node) {
  if (d.node_job_count[node] > 0) {
    push_node(d, node);
    return;
  }
  __threadfence();
  if (d.node_publish && d.node_publish[node] >= 0) {
    __threadfence_system();
    asm volatile("st.release.sys.global.u32 [%0], %1;" ::"l"(d.my_flags + d.node_publish[node]), "r"(d.epoch) : "memory");
  }
  for (int e = d.succ_off[node]; e < d.succ_off[node + 1]; ++e)
    if (atomicSub(&d.node_deps[d.succ[e]], 1) == 1) push_node(d, d.succ[e]);  // never job-less (builder)
  if (atomicAdd(d.done_nodes, 1) == d.total_nodes - 1) {
    __threadfence();
    atomicExch(d.finished, 1);
  }
}

// One warp pops one job: lanes inspect 32 queues at a time, highest priority first
// (two passes over the kBuckets buckets of the worker's class); the head node of the
// best non-empty queue hands out its next job; an exhausted head node is retired by
// advancing the queue head.  Returns -1 if nothing is ready.
__device__ __forceinline__ int try_pop(const DevSched& d, bool latency_worker, int lane, uint32_t done_bar,
                                       uint32_t done_parity) {
  const int cls = (d.policy == 2 && latency_worker) ? kBuckets : 0;  // pinned queues or normal ones
  bool gave_up = false;
  for (int pass = 0; pass < kBuckets / 32; ++pass) {
    const int q = cls + (kBuckets - 1 - (pass * 32 + lane));
    for (int attempt = 0; attempt < 16; ++attempt) {
      // the worker's running job finished: return to retire it (its successors may be
      // on the critical path) instead of racing other workers for queue heads
      if (done_bar && __any_sync(0xffffffffu, mbar_test_wait(done_bar, done_parity))) return -2;
      const int h = ld_volatile(&d.q_head[q * kQStride]);
      const int t = ld_volatile(&d.q_tail[q * kQStride]);
      const int item = h < t ? ld_volatile(&d.q_items[d.q_base[q] + h]) : 0;
      const unsigned m = __ballot_sync(0xffffffffu, item != 0);
      if (!m) break;
      const int src = __ffs(m) - 1;
      int job = -1;
      if (lane == src) {
        const int node = item - 1;
        const int j = atomicAdd(&d.node_next[node], 1);
        const int cnt = d.node_job_count[node];
        if (j < cnt) {
          job = d.node_job_begin[node] + j;
          // the claimer of a node's last job retires it from the head at once: lazy
          // retirement by later scanners walks claimed single-job nodes one CAS at a time
          if (j == cnt - 1) atomicCAS(&d.q_head[q * kQStride], h, h + 1);
        } else {
          atomicCAS(&d.q_head[q * kQStride], h, h + 1);  // node exhausted: retire it
          job = -2;
        }
      }
      job = __shfl_sync(0xffffffffu, job, src);
      if (job >= 0) return job;
      if (attempt == 15) gave_up = true;
    }
  }
  return gave_up ? -2 : -1;
}

// ------------------------------------------------------------------ warp-specialised worker
// CTA = 12 warps: warps 0-7 compute (setmaxnreg 232), warp 8 = TMA producer,
// warp 9 = scheduler, warp 10 = multi-GPU / streamed-input watcher (CTA 0), warp 11 = TMA-store
// epilogue (storer); control warpgroup at setmaxnreg 40.
// The scheduler pops the next job while the current one computes and does the
// completion bookkeeping off the compute warps; the producer walks the same job
// sequence through a 2-deep shared-memory job ring and issues every TMA load,
// running ahead into the next job as soon as ring stages free up.
// idle scheduler warp: exponential __nanosleep backoff up to this many ns (A/B via -D)
#ifndef CHOL_SCHED_BACKOFF_MAX
#define CHOL_SCHED_BACKOFF_MAX 256
#endif
constexpr int kWsThreads = 384;
constexpr int kProdWarp = 8, kSchedWarp = 9, kStoreWarp = 11;
constexpr int kRegsCompute = 232, kRegsControl = 40;

__device__ __forceinline__ void write_desc(int4* slot, int job, const Job& jb, int skip) {
  slot[0] = make_int4(job, (int)jb.type | (skip << 8), jb.i, jb.j);
  slot[1] = make_int4(jb.k, jb.a, jb.b, jb.c);
}

// ---- producer (one lane): issue the stages of a job, in the order the compute warps consume them
template <int BS>
__device__ __forceinline__ void produce_range(Ctx<BS>& c, uint32_t& pit, int nst, int64_t ta, int ra, int64_t tb,
                                              int rb, int kbeg, int from, int to) {
  for (int s = from; s < to && s < nst; ++s) issue_stage(c, pit + s, ta, ra, tb, rb, kbeg + s * BK);
}

// Jobs whose TMA loads the producer has finished issuing (shared memory, read by the
// scheduler warp): the scheduler claims job q+1 only once job q is fully issued, so a
// freshly enqueued critical job waits behind at most the tail of a running job.
__device__ __forceinline__ int* prod_issued_ptr(int4* jdesc) { return reinterpret_cast<int*>(jdesc + 6); }

// The BS x BS output block (store tile, row, column) a K-loop job updates: the C block the
// producer prefetches into lbuf and the storer writes back.  J_UPD / J_PUPD / J_TU.
template <int BS>
__device__ __forceinline__ void job_cblock(const Ctx<BS>& c, int type, const int4& d0, const int4& d1, int64_t* t,
                                           int* r0, int* c0) {
  if (type == J_UPD) {
    *t = c.slot(d0.z, d0.w), *r0 = d1.y * BS, *c0 = d1.z * BS;
  } else if (type == J_PUPD) {
    *t = c.slot(d1.x, d1.x), *r0 = d1.z * BS, *c0 = d1.w * BS;
  } else if (type == J_TU) {
    *t = c.slot(d0.z, d1.x), *r0 = d1.z * BS, *c0 = d1.w * BS;
  } else {  // J_TS: block (sl, cb) of A_ik
    *t = c.slot(d0.z, d1.x), *r0 = d1.z * BS, *c0 = d1.y * BS;
  }
}
__device__ __forceinline__ bool tma_store_job(int type) {
  return type == J_UPD || type == J_PUPD || type == J_TU || type == J_TS;
}

template <int BS>
__device__ void producer_loop(Ctx<BS>& c, const CUtensorMap* dmap) {
  uint32_t q = 0, pit = 0, tcount = 0, scount = 0;
  volatile int* issued = prod_issued_ptr(c.jdesc());
  while (true) {
    const int e = q & 1;
    mbar_wait(&c.jfull()[e], (q >> 1) & 1);
    const int4 d0 = c.jdesc()[e * 3], d1 = c.jdesc()[e * 3 + 1];
    const int job = d0.x, type = d0.y & 0xff, skip = d0.y >> 8;
    if (job < 0) break;
    fence_proxy_async();  // operands written by generic stores (this or other SMs)
    if (!skip) {
      const bool fused_diag = type == J_DIAG && d1.z;  // D(b) with U(b,b,b-1) in front
      if (type == J_UPD || type == J_PUPD || type == J_TU || fused_diag) {
        int64_t ta, tb, tcb;
        int ra, rb, kb, nst, cr, cc;
        if (fused_diag) {  // the update of block (b, b) by L[b, b-1] (k, b)
          ta = tb = tcb = c.slot(d1.x, d1.x);
          ra = rb = cr = cc = d1.y * BS;
          kb = (d1.y - 1) * BS;
          nst = BS / BK;
        } else if (type == J_UPD) {  // GEMM/SYRK block (i, j, k, bm, bn)
          ta = c.slot(d0.z, d1.x); ra = d1.y * BS;
          tb = c.slot(d0.w, d1.x); rb = d1.z * BS;
          kb = 0; nst = c.nb / BK;
          job_cblock(c, type, d0, d1, &tcb, &cr, &cc);
        } else if (type == J_PUPD) {  // POTRF update block (k, b, r, q)
          ta = tb = c.slot(d1.x, d1.x);
          ra = d1.z * BS; rb = d1.w * BS; kb = d1.y * BS; nst = BS / BK;
          job_cblock(c, type, d0, d1, &tcb, &cr, &cc);
        } else {  // TRSM update (i, k, c, s, c'): A_ik[s, c'] -= A_ik[s, c] L_kk[c', c]^T
          ta = c.slot(d0.z, d1.x);
          tb = c.slot(d1.x, d1.x);
          ra = d1.z * BS; rb = d1.w * BS; kb = d1.y * BS; nst = BS / BK;
          job_cblock(c, type, d0, d1, &tcb, &cr, &cc);
        }
        // the K-loop jobs add -acc to C with TMA reduce-add stores (no C block read);
        // the fused D(b) update keeps the C prefetch: stages first (they only need ring
        // space), then the C prefetch into lbuf once the previous job released it
        produce_range(c, pit, nst, ta, ra, tb, rb, kb, 0, kStages);
        if (fused_diag) {
          if (q > 0) mbar_wait(c.lfree(), (q - 1) & 1);
          prefetch_c_issue(c, tcb, cr, cc);
        }
        produce_range(c, pit, nst, ta, ra, tb, rb, kb, kStages, nst);
        pit += nst;
      } else if (type == J_TS) {
        // TS(cb, sl), inverse form: A_ik[sl, cb] Dinv_{k,cb}^T, K = BS -- A stages from the
        // tile store, B stages from the Dinv workspace; no C block (the result overwrites)
        const int64_t ta = c.slot(d0.z, d1.x);
        const int nbb = c.nb / BS, k = d1.x, cb = d1.y, ra = d1.z * BS;
        for (int s2 = 0; s2 < BS / BK; ++s2)
          issue_stage_ab(c, pit + s2, c.map, ta, ra, cb * BS + s2 * BK, dmap, k * nbb + cb, 0, s2 * BK);
        pit += BS / BK;
      } else if (type == J_TRSM) {
        // row slab (i, k, sl), inverse form; per column block cb: (1) cb*BS/BK stages of
        // X[sl, :cb] (solved) x L_kk[cb, :cb] -- the chunks of blocks solved before cb-1 are
        // final already and stream while the compute warps still work on block cb-1, the
        // last BS/BK wait for its write-back (tstep, from the storer); (2) X[sl, cb] into
        // lbuf once the previous staged block has been read (sfree; lfree of the previous
        // job for cb = 0); (3) BS/BK B-only stages of Dinv_{k,cb} (the A operand, Y, is
        // staged in lbuf).  The C prefetch precedes (3): the compute warps need it to form Y
        // before they can free the ring slots (3) waits for.
        const int nbb = c.nb / BS, k = d1.x;
        const int64_t ta = c.slot(d0.z, k), tb = c.slot(k, k);
        const int ra = d1.y * BS;
        for (int cb = 0; cb < nbb; ++cb) {
          if (cb > 0) {
            const int nst = cb * BS / BK, nold = (cb - 1) * BS / BK;
            produce_range(c, pit, nst, ta, ra, tb, cb * BS, 0, 0, nold);
            mbar_wait(c.tstep(), tcount & 1);
            ++tcount;
            fence_proxy_async();
            produce_range(c, pit, nst, ta, ra, tb, cb * BS, 0, nold, nst);
            pit += nst;
            mbar_wait(c.sfree(), scount & 1);
            ++scount;
          } else if (q > 0) {
            mbar_wait(c.lfree(), (q - 1) & 1);
          }
          prefetch_c_issue(c, ta, ra, cb * BS);
          for (int s2 = 0; s2 < BS / BK; ++s2) issue_stage_b(c, pit + s2, dmap, k * nbb + cb, s2 * BK);
          pit += BS / BK;
        }
      }
    }
    ++q;
    // jobs without TMA stages (in-register solves, POTRF diagonal blocks, RECV copies)
    // never mark themselves issued: their worker claims its next job only when they end,
    // so a critical job is not captured by a worker busy for another 10-20 us
    if (!skip && (type == J_UPD || type == J_PUPD || type == J_TU || type == J_TRSM || type == J_TS)) *issued = (int)q;
  }
}

// ---- storer (warp 11, one lane): the TMA-store epilogue of the K-loop jobs.  The compute
// warps stage -acc in lbuf (epi_stage_neg), arrive on cready and go on with their next
// job; the storer writes the block back with TMA (the same boxes the producer prefetched),
// releases lbuf once the store has read it (lfree) and completes the job (jdone) once the
// store has been performed -- only then does the scheduler warp release the successors.
// For every other job it just adds its arrival to lfree and jdone (both count compute
// warps + 1), after the previous job's lfree phase so its arrivals never run ahead.
template <int BS>
__device__ void storer_loop(Ctx<BS>& c) {
  uint32_t q = 0, ns = 0;
  while (true) {
    const int e = q & 1;
    mbar_wait(&c.jfull()[e], (q >> 1) & 1);
    const int4 d0 = c.jdesc()[e * 3], d1 = c.jdesc()[e * 3 + 1];
    const int job = d0.x, type = d0.y & 0xff, skip = d0.y >> 8;
    if (job < 0) break;
    if (q > 0) mbar_wait(c.lfree(), (q - 1) & 1);
    if (!skip && tma_store_job(type)) {
      int64_t t;
      int r0, c0;
      job_cblock(c, type, d0, d1, &t, &r0, &c0);
      mbar_wait(c.cready(), ns & 1);
      ++ns;
      const char* src = reinterpret_cast<const char*>(c.lbuf());
      if (type == J_TS) {  // overwrite
#pragma unroll 1
        for (int b = 0; b < BS / 16; ++b) tma_store_3d(c.map, src + b * BS * 128, c0 + 16 * b, r0, (int)t);
      } else {  // C += -acc
#pragma unroll 1
        for (int b = 0; b < BS / 16; ++b) tma_reduce_add_3d(c.map, src + b * BS * 128, c0 + 16 * b, r0, (int)t);
      }
      bulk_commit();
      bulk_wait_read_all();
      mbar_arrive(c.lfree());
      bulk_wait_all();
      fence_proxy_async();  // the async-proxy global writes before the generic release below
      __threadfence();
    } else if (!skip && type == J_TRSM) {
      // every solved column block Z_cb of the row slab: written back in place, then the
      // producer may stream it (tstep) as the last K chunk of block cb+1
      const int nbb = c.nb / BS;
      const int64_t t = c.slot(d0.z, d1.x);
      const int r0 = d1.y * BS;
      const char* src = reinterpret_cast<const char*>(c.lbuf());
      for (int cb = 0; cb < nbb; ++cb) {
        mbar_wait(c.cready(), ns & 1);
        ++ns;
#pragma unroll 1
        for (int b = 0; b < BS / 16; ++b) tma_store_3d(c.map, src + b * BS * 128, cb * BS + 16 * b, r0, (int)t);
        bulk_commit();
        bulk_wait_read_all();
        mbar_arrive(cb + 1 < nbb ? c.sfree() : c.lfree());
        bulk_wait_all();
        fence_proxy_async();
        __threadfence();
        if (cb + 1 < nbb) mbar_arrive(c.tstep());
      }
    } else {
      mbar_arrive(c.lfree());
    }
    mbar_arrive(&c.jdone()[e]);
    ++q;
  }
}

// ---- multi-GPU receive: row slab sl of remote panel tile (i, j) (BS rows x nb, contiguous:
// 737 KB at nb = 960), peer memory (NVLink) -> this rank's cache slot, by the TMA engine:
// thread 0 streams it through the two halves of lbuf with 1-D bulk copies -- peer -> shared
// (completion on rbar[h]), shared -> local global (bulk group) -- the load of chunk c+1
// overlapping the store of chunk c; the compute warps wait at the end.  The stores are
// complete and fenced before the job ends (its successors read the cache slot).
template <int BS>
__device__ __forceinline__ void recv_slab(Ctx<BS>& c, const DevSched& d, int i, int j, int sl, int owner) {
  if (threadIdx.x == 0) {
    const int64_t t = tile_index(i, j);
    const int64_t tile_elems = (int64_t)c.nb * c.nb, off = (int64_t)sl * BS * c.nb;
    const char* src = reinterpret_cast<const char*>(d.peer_slots[owner] + (int64_t)d.owner_slot[t] * tile_elems + off);
    char* dst = reinterpret_cast<char*>(c.tiles + c.slot(i, j) * tile_elems + off);
    char* buf = reinterpret_cast<char*>(c.lbuf());
    constexpr uint32_t kHalf = (Cfg<BS>::kBufBytes / 2) & ~1023u;  // bytes per chunk
    const int64_t total = (int64_t)BS * c.nb * 8;
    const int nch = (int)((total + kHalf - 1) / kHalf);
    auto load = [&](int ch) {
      const int64_t left = total - (int64_t)ch * kHalf;
      const uint32_t bytes = (uint32_t)(left < kHalf ? left : kHalf);
      uint64_t* bar = &c.rbar()[ch & 1];
      mbar_arrive_expect_tx(bar, bytes);
      bulk_load(buf + (ch & 1) * kHalf, src + (int64_t)ch * kHalf, bytes, bar);
    };
    fence_proxy_async();
    load(0);
    for (int ch = 0; ch < nch; ++ch) {
      const int64_t left = total - (int64_t)ch * kHalf;
      const uint32_t bytes = (uint32_t)(left < kHalf ? left : kHalf);
      if (ch + 1 < nch) {
        if (ch >= 1) bulk_wait_read<0>();  // buffer (ch+1)&1 = (ch-1)&1: its store has read it
        load(ch + 1);
      }
      // chunk ch landed (bit h of rcount: parity of the next completion of rbar[h])
      const int h = ch & 1;
      mbar_wait(&c.rbar()[h], (c.rcount >> h) & 1u);
      c.rcount ^= 1u << h;
      bulk_store(dst + (int64_t)ch * kHalf, buf + (ch & 1) * kHalf, bytes);
      bulk_commit();
    }
    bulk_wait_all();
    fence_proxy_async();
    __threadfence();
  }
  bar_sync(kBarCompute, kComputeThreads);
}

// ---- multi-GPU watcher (warp 10 of CTA 0): fires the RECV nodes whose remote tile became
// final (owner's flag == epoch), in step order, with a 64-entry sliding window.
__device__ void watcher_loop(const DevSched& d) {
  const int lane = threadIdx.x & 31;
  int w0 = 0;
  unsigned backoff = 64;
  while (w0 < d.nwatch && !ld_volatile(d.abort_flag)) {
    bool fired_any = false;
#pragma unroll
    for (int h = 0; h < 2; ++h) {
      const int e = w0 + h * 32 + lane;
      bool fire = false;
      int4 w = make_int4(0, 0, 0, 0);
      if (e < d.nwatch && !ld_volatile(&d.watch_fired[e])) {
        w = d.watch[e];
        unsigned f;
        asm volatile("ld.acquire.sys.global.u32 %0, [%1];" : "=r"(f) : "l"(d.peer_flags[w.y] + w.z) : "memory");
        fire = (f == d.epoch);
      }
      if (fire) {
        d.watch_fired[e] = 1;
        __threadfence();
        if (atomicSub(&d.node_deps[w.x], 1) == 1) ready_node(d, w.x);
      }
      fired_any |= __any_sync(0xffffffffu, fire);
    }
    // advance past the fired prefix
    while (true) {
      const int e = w0 + lane;
      const bool f = e >= d.nwatch || ld_volatile(&d.watch_fired[e]);
      const unsigned m = __ballot_sync(0xffffffffu, f);
      const int adv = (m == 0xffffffffu) ? 32 : __ffs(~m) - 1;
      w0 += adv;
      if (adv < 32 || w0 >= d.nwatch) break;
    }
    if (!fired_any) {
      __nanosleep(backoff);
      backoff = backoff < 1024 ? backoff * 2 : 1024;
    } else {
      backoff = 64;
    }
  }
}

// ---- development instrumentation (build with -DCHOL_PHASES, tools/job_phases.sh): warp 0
// of every CTA accumulates clock64 phases of the K = nb GEMM/SYRK block jobs -- [0] wait for
// the job descriptor, [1] job start -> first stage full, [2] mainloop, [3] epilogue,
// [4] epilogue end -> next descriptor wait, [5] job count; printed by chol_destroy.
#ifdef CHOL_PHASES
__device__ unsigned long long g_phase[8];
__device__ __forceinline__ long long phase_clock() { return clock64(); }
#define PHASE_ADD(i, v) \
  if (threadIdx.x == 0) atomicAdd(&g_phase[i], (unsigned long long)(v))
// TRSM row-slab jobs, per column block (warp 0): [0] Y mainloop (issue), [1] drain of its DMMA
// queue, [2] Y mainloop + stage_y, [3] Z mainloop, [4] stage_z, [5] blocks, [6] block 1's Y
__device__ unsigned long long g_tphase[8];
#define TPHASE_ADD(i, v) \
  if (threadIdx.x == 0) atomicAdd(&g_tphase[i], (unsigned long long)(v))
#else
#define PHASE_ADD(i, v)
#endif
void sched_phase_dump() {
#ifdef CHOL_HOPS
  {
    unsigned long long h[8];
    cudaMemcpyFromSymbol(h, g_hop, sizeof(h));
    const double nh = h[5] ? (double)h[5] : 1.0;
    fprintf(stderr, "CHOL_HOPS handoffs %llu  cycles: node_left %.0f  succ %.0f  pushes %.0f  count/trace %.0f  "
            "claim %.0f  (compute end -> jdone seen %.0f ns)\n", h[5], h[0] / nh, h[1] / nh, h[2] / nh, h[3] / nh,
            h[4] / nh, h[6] / nh);
    const unsigned long long z[8] = {};
    cudaMemcpyToSymbol(g_hop, z, sizeof(z));
  }
#endif
#ifdef CHOL_PHASES
  unsigned long long h[8];
  cudaMemcpyFromSymbol(h, g_phase, sizeof(h));
  const double nj = h[5] ? (double)h[5] : 1.0;
  fprintf(stderr, "CHOL_PHASES jobs %llu  cycles/job: wait_desc %.0f  first_stage %.0f  mainloop %.0f  epilogue %.0f  "
          "to_next %.0f  (drain of the DMMA queue, inside epilogue: %.0f)\n", h[5], h[0] / nj, h[1] / nj, h[2] / nj,
          h[3] / nj, h[4] / nj, h[6] / nj);
  const unsigned long long z[8] = {};
  cudaMemcpyToSymbol(g_phase, z, sizeof(z));
  unsigned long long tp[8];
  cudaMemcpyFromSymbol(tp, g_tphase, sizeof(tp));
  const double nbk = tp[5] ? (double)tp[5] : 1.0;
  fprintf(stderr, "CHOL_PHASES trsm blocks %llu  cycles/block: Y mainloop %.0f (drain %.0f)  Y+stage_y %.0f  Z %.0f  "
          "stage_z %.0f  block-1 Y %.0f\n", tp[5], tp[0] / nbk, tp[1] / nbk, tp[2] / nbk, tp[3] / nbk, tp[4] / nbk,
          tp[6] / (nbk / 10.0));
  cudaMemcpyToSymbol(g_tphase, z, sizeof(z));
#endif
}

// ---- compute warps: run the job's consumer side
template <int BS>
__device__ __forceinline__ void compute_job(Ctx<BS>& c, const DevSched& d, int type, uint32_t q, const int4& d0,
                                            const int4& d1,
                                            int* info) {
  // accumulators are declared per branch: one function-wide Acc makes ptxas keep its
  // registers reserved across the register-hungry in-block routines (spills)
  if (type == J_UPD) {
    Acc<BS> acc;
    const int i = d0.z, j = d0.w, k = d1.x, bm = d1.y, bn = d1.z;
#ifdef CHOL_PHASES
    const long long p0 = phase_clock();
    mbar_wait(&c.full()[c.it % kStages], (c.it / kStages) & 1);
    const long long p1 = phase_clock();
#endif
    gemm_consume(c, c.nb / BK, acc);
#ifdef CHOL_PHASES
    const long long p2 = phase_clock();
    {  // wait for the last-issued DMMA (its accumulator) -> drain of the DMMA queue
      volatile double sink = acc[Cfg<BS>::MI - 1][Cfg<BS>::NI - 1][1] + acc[0][0][0];
      (void)sink;
      PHASE_ADD(6, phase_clock() - p2);
    }
#endif
    if (q > 0) mbar_wait(c.lfree(), (q - 1) & 1);  // the previous job's staged block has been read
    epi_stage_neg(c, acc, i == j && bm == bn);
#ifdef CHOL_PHASES
    const long long p3 = phase_clock();
    PHASE_ADD(1, p1 - p0);
    PHASE_ADD(2, p2 - p1);
    PHASE_ADD(3, p3 - p2);
    PHASE_ADD(5, 1);
#endif
    (void)k;
  } else if (type == J_PUPD) {
    Acc<BS> acc;
    const int r = d1.z, qb = d1.w;
    gemm_consume(c, BS / BK, acc);
    if (q > 0) mbar_wait(c.lfree(), (q - 1) & 1);
    epi_stage_neg(c, acc, r == qb);
  } else if (type == J_TRSM) {
    // row slab X = A_ik[sl, :] <- X L_kk^{-T} (L200-202), left-looking over the BS-column
    // blocks, inverse form (reading R19): Y = X[:, cb] - X[:, :cb] L_kk[cb, :cb]^T, then
    // X[:, cb] = Y Dinv_cb^T -- two DMMA products per block, no in-block substitution
    const int i = d0.z, k = d1.x, slab = d1.y, nbb = c.nb / BS;
    prefetch_l2_rows<BS>(c.tile(i, k) + (int64_t)slab * BS * c.nb, c.nb, BS, c.nb);
    for (int cb = 0; cb < nbb; ++cb) {
#ifdef CHOL_PHASES
      const long long q0 = phase_clock();
#endif
      {
        Acc<BS> acc;
        gemm_consume(c, cb * BS / BK, acc);  // zero for cb = 0
#ifdef CHOL_PHASES
        const long long q1 = phase_clock();
        TPHASE_ADD(0, q1 - q0);
        {
          volatile double sink = acc[Cfg<BS>::MI - 1][Cfg<BS>::NI - 1][1] + acc[0][0][0];
          (void)sink;
        }
        const long long q2 = phase_clock();
        TPHASE_ADD(1, q2 - q1);
#endif
        trsm_stage_y(c, acc);
      }
#ifdef CHOL_PHASES
      const long long q3 = phase_clock();
#endif
      Acc<BS> z;
      gemm_consume<BS, true>(c, BS / BK, z);
#ifdef CHOL_PHASES
      const long long q4 = phase_clock();
#endif
      trsm_stage_z(c, z);
      __syncwarp();
      if (c.lane == 0) mbar_arrive(c.cready());  // the storer writes Z_cb back
#ifdef CHOL_PHASES
      const long long q5 = phase_clock();
      TPHASE_ADD(2, q3 - q0);
      TPHASE_ADD(3, q4 - q3);
      TPHASE_ADD(4, q5 - q4);
      if (cb == 1) TPHASE_ADD(6, q3 - q0);
      TPHASE_ADD(5, 1);
#endif
    }
  } else if (type == J_INV) {
    const int k = d1.x, b = d1.y, nbb = c.nb / BS;
    inv_block_job<BS>(c.tile(k, k) + (int64_t)b * BS * c.nb + b * BS, c.nb,
                      d.dinv + ((int64_t)k * nbb + b) * BS * BS);
  } else if (type == J_TU) {
    Acc<BS> acc;
    gemm_consume(c, BS / BK, acc);
    if (q > 0) mbar_wait(c.lfree(), (q - 1) & 1);
    epi_stage_neg(c, acc, false);
  } else if (type == J_TS) {  // X[sl, cb] <- X[sl, cb] Dinv_{k,cb}^T (inverse form, reading R19)
    Acc<BS> z;
    gemm_consume(c, BS / BK, z);
    trsm_stage_z(c, z);  // the storer writes it back
  } else if (type == J_RECV) {  // copy BS rows of a remote panel tile into the local cache
    const int i = d0.z, j = d0.w, sl = d1.y, owner = d1.z;
    (void)owner;
    recv_slab(c, d, i, j, sl, owner);
  } else if (type == J_DIAG) {
    if (d1.z) {  // fused U(b,b,b-1): the K = BS update of the block first, same code as J_PUPD
      Acc<BS> acc;
      const int k = d1.x, b = d1.y;
      gemm_consume(c, BS / BK, acc);
      epi_sub_global(c, acc, c.tile(k, k) + (int64_t)b * BS * c.nb + b * BS, c.nb, true);
    }
    sub_potrf_diag(c, d1.x, d1.y, info);  // its first barrier orders the stores above
  } else if (type == J_PANEL) {
    sub_potrf_panel(c, d1.x, d1.y, d1.z);
  }
}

template <int BS>
__device__ void compute_loop(Ctx<BS>& c, const DevSched& d, int* info) {
  uint32_t q = 0;
#ifdef CHOL_PHASES
  long long t_end = 0;
  bool last_upd = false;
#endif
  while (true) {
    const int e = q & 1;
#ifdef CHOL_PHASES
    const long long w0 = phase_clock();
#endif
    mbar_wait(&c.jfull()[e], (q >> 1) & 1);
#ifdef CHOL_PHASES
    if (last_upd) {
      PHASE_ADD(0, phase_clock() - w0);
      PHASE_ADD(4, w0 - t_end);
    }
#endif
    const int4 d0 = c.jdesc()[e * 3], d1 = c.jdesc()[e * 3 + 1];
    if (d0.x < 0) break;
    if (c.warp == 0 && c.lane == 0) {
      const unsigned long long t0 = globaltimer_ns();
      c.jdesc()[e * 3 + 2] = make_int4((int)(t0 & 0xffffffffull), (int)(t0 >> 32), 0, 0);
    }
    const int type = d0.y & 0xff, skip = d0.y >> 8;
    // jobs that use lbuf directly (in-block solves, potf2, the fused update's C block is
    // prefetched behind lfree anyway) wait until the previous job's TMA store has read it
    if (!skip && q > 0 && (type == J_INV || type == J_TS || type == J_PANEL || type == J_DIAG || type == J_RECV))
      mbar_wait(c.lfree(), (q - 1) & 1);
    if (!skip) compute_job(c, d, type, q, d0, d1, info);
    if (!skip && tma_store_job(type)) {
      __syncwarp();
      if (c.lane == 0) mbar_arrive(c.cready());  // C - acc staged: the storer takes over
    }
#ifdef CHOL_PHASES
    last_upd = !skip && type == J_UPD;
#endif
    __syncwarp();
    if (c.lane == 0) {
      // lfree has one phase per job (compute warps + the storer): a job that ends quickly
      // (skipped after a failed pivot, no lbuf use) must not arrive into the previous
      // job's phase while the storer is still reading that job's staged block
      if (q > 0) mbar_wait(c.lfree(), (q - 1) & 1);
      mbar_arrive(c.lfree());  // lbuf (C block / L block / rdiag) no longer needed
      if (c.warp == 0) {     // end time of the job as seen by warp 0
        const unsigned long long t1 = globaltimer_ns();
        c.jdesc()[e * 3 + 2].z = (int)(t1 & 0xffffffffull);
        c.jdesc()[e * 3 + 2].w = (int)(t1 >> 32);
      }
      mbar_arrive(&c.jdone()[e]);  // the job's global stores precede this release
    }
    ++q;
#ifdef CHOL_PHASES
    t_end = phase_clock();
#endif
  }
}

// Trace records of a completed job (after the releases: every job of a task updates the
// same two words, and that contention must not delay the successors).
__device__ __forceinline__ void trace_job(const DevSched& d, const StepParams& sp, int node, int job, uint64_t t0_abs,
                                          uint64_t t1_abs, int lane) {
  if (lane == 0 && sp.tr_t0 && d.node_paper[node] >= 0) {
    const uint64_t base = *sp.tr_base;
    const uint64_t t0 = t0_abs - base, t_end = t1_abs - base;
    const int pt = d.node_paper[node];
    atomicMin(reinterpret_cast<unsigned long long*>(sp.tr_t0 + pt), (unsigned long long)t0);
    atomicMax(reinterpret_cast<unsigned long long*>(sp.tr_t1 + pt), (unsigned long long)((t_end << 16) | smid()));
    if (d.job_trace) {
      d.job_trace[4 * (size_t)job] = t0;
      d.job_trace[4 * (size_t)job + 1] = t_end;
      d.job_trace[4 * (size_t)job + 2] = ((uint64_t)blockIdx.x << 32) | smid();
    }
  }
}

// ---- hand-off fast path.  While a job runs alone on its worker, the scheduler warp
// preloads the successor list of the job's node into shared memory: successor ids, their
// job counts and, for single-job successors, the job descriptor (all of these tables are
// constant during a launch).  At completion the successors are released with one round of
// atomics and a ready single-job successor is written into the job ring straight from the
// preloaded descriptor, before the other successors are queued and the node is counted --
// none of the dependent global loads of the generic path (node, successor list, job count,
// job begin, descriptor) are left between the end of one job and the start of the next on
// a chain of single-job nodes (the POTRF block DAG's D(b) -> P(b+1,b) -> D(b+1)).
struct SuccPre {
  int4 sjob[32];                   // Job of single-job successor l (raw 16 bytes)
  int succ[32], scnt[32], sbeg[32];
  int job, node, jc, ns;           // preloaded job (-1: none), its node, job count, successors
};
static_assert(sizeof(Job) == 16, "Job is loaded as one int4");

#ifndef CHOL_PRE_MODE
#define CHOL_PRE_MODE 2  // development switch: 0 no preload, 1 after claims only, 2 also while idle
#endif
__device__ __forceinline__ void fence_acq_rel_gpu() { asm volatile("fence.acq_rel.gpu;" ::: "memory"); }

__device__ void preload_succ(const DevSched& d, SuccPre* P, int job, int lane) {
  const int node = __ldg(d.job_node + job);
  const int beg = __ldg(d.succ_off + node), ns = __ldg(d.succ_off + node + 1) - beg;
  int sc = 1;
  if (lane < ns) {
    const int sn = __ldg(d.succ + beg + lane);
    sc = __ldg(d.node_job_count + sn);
    const int sb = __ldg(d.node_job_begin + sn);
    P->succ[lane] = sn;
    P->scnt[lane] = sc;
    P->sbeg[lane] = sb;
    if (sc == 1) P->sjob[lane] = __ldg(reinterpret_cast<const int4*>(d.jobs) + sb);
  }
  // a node with more than 32 successors or a job-less successor keeps the generic path
  const bool ok = ns <= 32 && __all_sync(0xffffffffu, sc > 0);
  if (lane == 0) {
    P->node = node;
    P->jc = __ldg(d.node_job_count + node);
    P->ns = ns;
    P->job = ok ? job : -2 - job;
  }
  __syncwarp();
}

// Completion of the preloaded job.  Returns the job written into the ring slot (slot /
// jfull_e: the next free entry) or -1.  Same releases and counts as complete_job +
// node_done_warp (the preloaded nodes have no job-less successor), hand-off first.
__device__ int complete_job_pre(const DevSched& d, const StepParams& sp, const SuccPre* P, uint64_t t0_abs,
                                uint64_t t1_abs, int lane, bool can_take, int4* slot, uint64_t* jfull_e) {
  const int node = P->node, job = P->job;
  int last = 1;
  if (P->jc != 1) {  // several jobs: the node is done when its counter runs out
    if (lane == 0) {
      __threadfence();  // the compute warps' stores (acquired through jdone) before the counter
      last = atomicSub(&d.node_left[node], 1) == 1;
    }
    last = __shfl_sync(0xffffffffu, last, 0);
  }
  HOP_MARK(3);
  int issued = -1;
  if (last) {
    fence_acq_rel_gpu();  // every job of the node (this worker's stores, the other jobs' releases) before the edges
    const int inf = ld_volatile(sp.info);
    const int ns = P->ns;
    int sn = -1, cnt = -1;
    if (lane < ns) {
      sn = P->succ[lane];
      if (atomicSub(&d.node_deps[sn], 1) == 1) cnt = P->scnt[lane];
    }
    const unsigned ms = __ballot_sync(0xffffffffu, can_take && cnt == 1);
    const int taker = ms ? __ffs(ms) - 1 : -1;
    if (taker >= 0) {
      HOP_MARK(0);
      if (lane == taker) {
        fence_acq_rel_gpu();  // acquire: the other predecessors' releases, before the job's loads
        const int4 raw = P->sjob[lane];
        const Job jb = *reinterpret_cast<const Job*>(&raw);
        const int jid = P->sbeg[lane];
        write_desc(slot, jid, jb, inf != INT_MAX && jb.k >= (inf - 1) / sp.nb);
        mbar_arrive(jfull_e);
        if (d.job_trace) d.job_trace[4 * (size_t)jid + 3] = globaltimer_ns() - *d.tr_base;
      }
      issued = P->sbeg[taker];
    }
    __syncwarp();
    HOP_MARK(1);
    publish_node(d, node, lane);
    if (cnt > 0 && lane != taker) push_node(d, sn);
    count_node_done(d, lane);
    HOP_MARK(2);
  }
  trace_job(d, sp, node, job, t0_abs, t1_abs, lane);
  return issued;
}

// ---- scheduler warp (all lanes): job counter, node completion, trace
__device__ __forceinline__ int complete_job(const DevSched& d, const StepParams& sp, int job, uint64_t t0_abs,
                                            uint64_t t1_abs, int lane, bool can_take) {
  const int node = d.job_node[job];
  int last = 0;
  if (lane == 0) {
    __threadfence();  // the compute warps' stores (acquired through jdone) before the counters
    last = atomicSub(&d.node_left[node], 1) == 1;
  }
  HOP_MARK(3);
  const int take = __shfl_sync(0xffffffffu, last, 0) ? node_done_warp<1>(d, node, lane, can_take) : -1;
  // trace records after the release: every job of a task updates the same two words,
  // and that contention must not delay the successors
  trace_job(d, sp, node, job, t0_abs, t1_abs, lane);
  return take;
}
template <int BS>
__device__ void scheduler_loop(Ctx<BS>& c, const DevSched& d, const StepParams& sp, bool latency_worker) {
  const int lane = c.lane;
  uint32_t q_issue = 0, q_done = 0;
  int pending[2] = {-1, -1};
  int take = -1;  // single-job successor handed to this worker by its own completion
  unsigned backoff = 32;
  SuccPre* P = reinterpret_cast<SuccPre*>(Ctx<BS>::pre());
  if (lane == 0) P->job = -1;
  __syncwarp();
#ifdef CHOL_HOPS
  long long h_claim_from = 0;
#endif
  while (true) {
    // 1. retire finished jobs in order
    while (q_done < q_issue) {
      const int e = q_done & 1;
      if (!mbar_try_wait(smem_u32(&c.jdone()[e]), (q_done >> 1) & 1)) break;
      HOP_T(h_seen);
#ifdef CHOL_HOPS
      const unsigned long long h_gt = globaltimer_ns();
#endif
      const int4 tt = c.jdesc()[e * 3 + 2];
      const uint64_t t0 = (uint64_t)(uint32_t)tt.x | ((uint64_t)(uint32_t)tt.y << 32);
      const uint64_t t1 = (uint64_t)(uint32_t)tt.z | ((uint64_t)(uint32_t)tt.w << 32);
      const bool can_take = take < 0 && q_done + 1 == q_issue;
      if (P->job == pending[e]) {  // successors preloaded: hand-off fast path
        const int ne = q_issue & 1;
        const int iss = complete_job_pre(d, sp, P, t0, t1, lane, can_take, &c.jdesc()[ne * 3], &c.jfull()[ne]);
#ifdef CHOL_HOPS
        HOP_T(h_ret);
        if (iss >= 0) {
          const long long* m = g_hopt[blockIdx.x];
          HOP_ADD(0, m[3] - h_seen);
          HOP_ADD(1, m[0] - m[3]);
          HOP_ADD(4, m[1] - m[0]);
          HOP_ADD(3, h_ret - m[1]);
          HOP_ADD(6, h_gt - t1);
          HOP_ADD(5, 1);
        }
#endif
        ++q_done;
        if (iss >= 0) {  // the successor is running already: preload its successors
          pending[ne] = iss;
          ++q_issue;
          backoff = 32;
          preload_succ(d, P, iss, lane);
        }
        continue;
      }
      const int t = complete_job(d, sp, pending[e], t0, t1, lane, can_take);
      if (t >= 0) take = t;
#ifdef CHOL_HOPS
      HOP_T(h_ret);
      if (t >= 0) {
        const long long* m = g_hopt[blockIdx.x];
        HOP_ADD(0, m[3] - h_seen);
        HOP_ADD(1, m[0] - m[3]);
        HOP_ADD(2, m[1] - m[0]);
        HOP_ADD(3, h_ret - m[1]);
        HOP_ADD(6, h_gt - t1);
      }
      h_claim_from = t >= 0 ? h_ret : 0;
#endif
      ++q_done;
    }
    // 2. claim the next job once the ring has room and the producer is done with the
    //    running job's loads (late claim keeps critical-path hops short)
    if (q_issue - q_done < 2 && (q_issue == q_done || ld_volatile(prod_issued_ptr(c.jdesc())) >= (int)q_issue)) {
      const int job = take >= 0 ? d.node_job_begin[take]
                                : try_pop(d, latency_worker, lane,
                                          q_issue > q_done ? smem_u32(&c.jdone()[q_done & 1]) : 0u, (q_done >> 1) & 1);
      take = -1;
      if (job >= 0) {
        const int e = q_issue & 1;
        if (lane == 0) {
          __threadfence();  // acquire: the job's inputs were published before it was enqueued
          const Job jb = d.jobs[job];
          // after a non-positive pivot in tile column kf = (info-1)/nb only the jobs of
          // steps >= kf are skipped: every job of an earlier step (TRSM_i_k, the updates
          // of step k < kf) still runs, so columns < kf*nb of L are final (chol.h, info)
          const int inf = ld_volatile(sp.info);
          write_desc(&c.jdesc()[e * 3], job, jb, inf != INT_MAX && jb.k >= (inf - 1) / sp.nb);
          mbar_arrive(&c.jfull()[e]);
#ifdef CHOL_HOPS
          if (h_claim_from) {
            atomicAdd(&g_hop[4], (unsigned long long)(clock64() - h_claim_from));
            atomicAdd(&g_hop[5], 1ull);
          }
#endif
        }
#ifdef CHOL_HOPS
        h_claim_from = 0;
#endif
        __syncwarp();
        pending[e] = job;
        ++q_issue;
        backoff = 32;
        if (CHOL_PRE_MODE >= 1 && q_issue == q_done + 1) preload_succ(d, P, job, lane);
        continue;
      }
    }
    // the job running alone (its successor list may be needed for a hand-off)
    if (CHOL_PRE_MODE >= 2 && q_issue == q_done + 1 && P->job != pending[q_done & 1] &&
        P->job != -2 - pending[q_done & 1]) {
      preload_succ(d, P, pending[q_done & 1], lane);
      continue;
    }
    // 3. done?
    if (q_done == q_issue && (ld_volatile(d.finished) || ld_volatile(d.abort_flag))) {
      if (lane == 0) {
        const int e = q_issue & 1;
        c.jdesc()[e * 3] = make_int4(-1, 0, 0, 0);
        mbar_arrive(&c.jfull()[e]);
      }
      __syncwarp();
      break;
    }
    __nanosleep(backoff);
    backoff = backoff < CHOL_SCHED_BACKOFF_MAX ? backoff * 2 : CHOL_SCHED_BACKOFF_MAX;
  }
}

template <int BS>
__global__ void __launch_bounds__(kWsThreads, 1) k_sched(const __grid_constant__ CUtensorMap map,
                                                         const __grid_constant__ CUtensorMap dmap, StepParams sp,
                                                         DevSched d) {
  auto c = make_ctx<BS>(&map, sp.tiles, sp.nb, sp.N, d.slot_map);
  const bool latency_worker = d.policy == 2 && (int)blockIdx.x < d.latency_workers;
  if (c.warp >= kComputeWarps) {
    asm volatile("setmaxnreg.dec.sync.aligned.u32 %0;\n" ::"n"(kRegsControl));
    if (c.warp == kProdWarp) {
      if (c.lane == 0) producer_loop(c, &dmap);
    } else if (c.warp == kSchedWarp) {
      scheduler_loop(c, d, sp, latency_worker);
    } else if (c.warp == kSchedWarp + 1 && blockIdx.x == 0 && d.nwatch > 0) {
      watcher_loop(d);
    } else if (c.warp == kStoreWarp) {
      if (c.lane == 0) storer_loop(c);
    }
    return;
  }
  asm volatile("setmaxnreg.inc.sync.aligned.u32 %0;\n" ::"n"(kRegsCompute));
  compute_loop(c, d, sp.info);
}

// Roots pushed in parallel (a calibration batch has up to ~1100 roots: one thread took
// 70 us); their order within a queue is a scheduling choice, never a numerical one (R15).
__global__ void k_sched_init(DevSched d, const int* roots, int nroots) {
  for (int r = blockIdx.x * blockDim.x + threadIdx.x; r < nroots; r += gridDim.x * blockDim.x)
    ready_node(d, roots[r]);
}

// ------------------------------------------------------------------ host planner
struct SchedState {
  int64_t N = 0, nb = 0;
  int arrival = 0;  // streamed-input tile order (arrival_order)
  int bs = 0, workers = 0, nnodes = 0, njobs = 0, nroots = 0;
  chol_opts_t opts{};
  DevSched d{};
  // device buffers
  void* dev_static = nullptr;   // jobs, job_node, CSR, node tables (read-only)
  void* dev_dynamic = nullptr;  // counters, queues (reset per run)
  size_t dyn_bytes = 0;
  void* dev_pristine = nullptr; // initial node_deps / node_left
  size_t pristine_bytes = 0;
  int* roots = nullptr;
  int nrecv_jobs = 0;
  uint64_t* job_trace = nullptr;           // device, 4 per job (trace == 2)
  int* d_abort = nullptr;                  // device abort flag (d.abort_flag), written by sched_abort
  CUtensorMap dmap{};                      // Dinv workspace map (sched_set_dinv)
  std::vector<std::pair<int, int>> host_tasks;  // TRSM_i_k run by the host CPU class (i, k)
  // re-bucketing with injected task priorities (sched_set_priorities)
  std::vector<int> h_node_paper, h_node_queue;
  size_t o_nq = 0, o_qbase = 0;
  std::vector<int16_t> h_job_type;         // host copies for chol_job_trace
  std::vector<Job> h_jobs;                 // ... and chol_job_desc
  std::vector<int> h_job_node;
  std::vector<int> h_job_paper;
};

namespace {

struct Builder {
  int64_t N;
  int nbb, policy, pin_d;
  std::vector<Job> jobs;
  std::vector<int> job_node, deps, jbeg, jcnt, paper, ptype, pk, pi;
  std::vector<std::vector<int>> succ;

  int add_node(int paper_id, int type, int i, int k) {
    const int id = (int)deps.size();
    deps.push_back(0);
    jbeg.push_back((int)jobs.size());
    jcnt.push_back(0);
    paper.push_back(paper_id);
    ptype.push_back(type);
    pi.push_back(i);
    pk.push_back(k);
    succ.emplace_back();
    return id;
  }
  void add_job(int node, Job j) {
    jobs.push_back(j);
    job_node.push_back(node);
    ++jcnt[node];
  }
  void edge(int a, int b) {
    succ[a].push_back(b);
    ++deps[b];
  }
};

}  // namespace

// POTRF_k as per-step nodes: DIAG b -> PANEL b (nbb-1-b jobs) -> UPDATE b (K = BS) -> DIAG b+1
static void build_potrf_steps(Builder& B, int k, int pid, int* first, int* last, std::vector<int>* dnodes = nullptr) {
  const int nbb = B.nbb;
  int prev = -1;
  if (dnodes) dnodes->assign(nbb, -1);
  for (int b = 0; b < nbb; ++b) {
    const int dn = B.add_node(pid, T_POTRF, k, k);
    B.add_job(dn, Job{J_DIAG, (int16_t)k, (int16_t)k, (int16_t)k, (int16_t)b, 0, 0, 0});
    if (dnodes) (*dnodes)[b] = dn;
    if (prev >= 0) B.edge(prev, dn);
    if (b == 0) *first = dn;
    prev = dn;
    if (b + 1 < nbb) {
      const int pn = B.add_node(pid, T_POTRF, k, k);
      for (int r = b + 1; r < nbb; ++r)
        B.add_job(pn, Job{J_PANEL, (int16_t)k, (int16_t)k, (int16_t)k, (int16_t)b, (int16_t)r, 0, 0});
      B.edge(prev, pn);
      const int un = B.add_node(pid, T_POTRF, k, k);
      for (int r = b + 1; r < nbb; ++r)
        for (int q = b + 1; q <= r; ++q)
          B.add_job(un, Job{J_PUPD, (int16_t)k, (int16_t)k, (int16_t)k, (int16_t)b, (int16_t)r, (int16_t)q, 0});
      B.edge(pn, un);
      prev = un;
    }
  }
  *last = prev;
}

// POTRF_k as a block-level DAG over the BS x BS blocks of the diagonal tile (right-looking
// nested Cholesky): D(b) = potf2 of block (b,b); P(r,b) = solve of block (r,b) against
// L_bb; U(r,q,b) = K=BS update of block (r,q) by blocks (r,b), (q,b).  One job per node, so
// the chain D(b) -> P(b+1,b) -> U(b+1,b+1,b) -> D(b+1) never waits for a whole column or
// trailing update of the step.  D(nbb-1) is the sink (every inner node is its ancestor).
// With fuse the chain's last update U(b,b,b-1) is done by D(b) itself: the job runs the
// J_PUPD code (producer stages, DMMA, epilogue) and then potf2 -- one node and one hop less
// per inner step, the same bits.  blk (hybrid tail): record per block the entry node and
// the node that leaves it final (tentry / tfin, nbb x nbb).
static void build_potrf_blockdag(Builder& B, int k, int pid, bool fuse, bool blk, std::vector<int>* tentry,
                                 std::vector<int>* tfin, int* first, int* last, std::vector<int>* dnodes = nullptr) {
  const int nbb = B.nbb;
  std::vector<int> lastU((size_t)nbb * nbb, -1), pan(nbb, -1), fusedP(nbb, -1);
  if (blk) tentry->assign((size_t)nbb * nbb, -1), tfin->assign((size_t)nbb * nbb, -1);
  if (dnodes) dnodes->assign(nbb, -1);
  for (int b = 0; b < nbb; ++b) {
    const int dn = B.add_node(pid, T_POTRF, k, k);
    B.add_job(dn, Job{J_DIAG, (int16_t)k, (int16_t)k, (int16_t)k, (int16_t)b, (int16_t)(fusedP[b] >= 0), 0, 0});
    if (dnodes) (*dnodes)[b] = dn;
    if (lastU[b * nbb + b] >= 0) B.edge(lastU[b * nbb + b], dn);
    if (fusedP[b] >= 0) B.edge(fusedP[b], dn);
    if (blk && b == 1 && fusedP[b] >= 0) (*tentry)[b * nbb + b] = dn;  // first touch of block (1,1)
    if (b == 0) *first = dn;
    *last = dn;
    for (int r = b + 1; r < nbb; ++r) {
      const int pn = B.add_node(pid, T_POTRF, k, k);
      B.add_job(pn, Job{J_PANEL, (int16_t)k, (int16_t)k, (int16_t)k, (int16_t)b, (int16_t)r, 0, 0});
      B.edge(dn, pn);
      if (lastU[r * nbb + b] >= 0) B.edge(lastU[r * nbb + b], pn);
      pan[r] = pn;
    }
    for (int r = b + 1; r < nbb; ++r)
      for (int q = b + 1; q <= r; ++q) {
        if (fuse && r == b + 1 && q == r) {  // U(b+1,b+1,b): fused into D(b+1)
          fusedP[r] = pan[r];
          continue;
        }
        const int un = B.add_node(pid, T_POTRF, k, k);
        B.add_job(un, Job{J_PUPD, (int16_t)k, (int16_t)k, (int16_t)k, (int16_t)b, (int16_t)r, (int16_t)q, 0});
        B.edge(pan[r], un);
        if (q != r) B.edge(pan[q], un);
        if (lastU[r * nbb + q] >= 0) B.edge(lastU[r * nbb + q], un);  // same block, previous step
        lastU[r * nbb + q] = un;
        if (blk && b == 0) (*tentry)[r * nbb + q] = un;
      }
    if (blk) {
      (*tfin)[b * nbb + b] = dn;
      if (b == 0) (*tentry)[0] = dn;
      for (int r = b + 1; r < nbb; ++r) {
        (*tfin)[r * nbb + b] = pan[r];
        if (b == 0) (*tentry)[r * nbb] = pan[r];
      }
    }
  }
}

// The inverses of the diagonal blocks of L_kk that the inverse-form TRSM row slabs of step k
// apply (J_TRSM): INV(k, b) after the node that makes block (b, b) of L_kk final (pred[b],
// or pred[0] alone for a received tile), a job-less join INVJ(k), and INVJ(k) -> every row
// slab node of step k.  Untraced (paper id -1, highest priority bucket: it gates TRSM work).
// The right-looking TS(cb, .) nodes (TRSM column-step solves, also inverse form) wait for
// INV(k, cb) alone: ts[cb] lists them.
static void build_inverses(Builder& B, int k, const std::vector<int>& pred, const std::vector<int>& slabs,
                           const std::vector<std::vector<int>>& ts = {}) {
  bool any_ts = false;
  for (const auto& v : ts) any_ts |= !v.empty();
  if (slabs.empty() && !any_ts) return;
  const int nbb = B.nbb;
  const int join = slabs.empty() ? -1 : B.add_node(-1, T_POTRF, k, k);
  for (int b = 0; b < nbb; ++b) {
    const int v = B.add_node(-1, T_POTRF, k, k);
    B.add_job(v, Job{J_INV, (int16_t)k, (int16_t)k, (int16_t)k, (int16_t)b, 0, 0, 0});
    const int p = pred.size() == (size_t)nbb ? pred[b] : (pred.empty() ? -1 : pred[0]);
    if (p >= 0) B.edge(p, v);
    if (join >= 0) B.edge(v, join);
    if (b < (int)ts.size())
      for (int t : ts[b]) B.edge(v, t);
  }
  for (int sn : slabs) B.edge(join, sn);
}

// TRSM_i_k right-looking over the BS-column blocks c of A_ik, one node per column step:
//   TS(c): A_ik[:, c] <- A_ik[:, c] L_kk[c,c]^{-T}  (nbb row-block jobs)
//   TU(c): A_ik[:, c'] -= A_ik[:, c] L_kk[c',c]^T, c' > c  (K = BS)
static void build_trsm_steps(Builder& B, int i, int k, int tid, int* first, int* last,
                             std::vector<std::vector<int>>* ts_nodes = nullptr) {
  const int nbb = B.nbb;
  int prev_t = -1;
  if (ts_nodes && ts_nodes->empty()) ts_nodes->resize(nbb);
  for (int cb = 0; cb < nbb; ++cb) {
    const int ts = B.add_node(tid, T_TRSM, i, k);
    if (ts_nodes) (*ts_nodes)[cb].push_back(ts);
    for (int sl = 0; sl < nbb; ++sl)
      B.add_job(ts, Job{J_TS, (int16_t)i, (int16_t)k, (int16_t)k, (int16_t)cb, (int16_t)sl, 0, 0});
    if (prev_t >= 0) B.edge(prev_t, ts);
    if (cb == 0) *first = ts;
    prev_t = ts;
    if (cb + 1 < nbb) {
      const int tu = B.add_node(tid, T_TRSM, i, k);
      for (int sl = 0; sl < nbb; ++sl)
        for (int c2 = cb + 1; c2 < nbb; ++c2)
          B.add_job(tu, Job{J_TU, (int16_t)i, (int16_t)k, (int16_t)k, (int16_t)cb, (int16_t)sl, (int16_t)c2, 0});
      B.edge(ts, tu);
      prev_t = tu;
    }
  }
  *last = prev_t;
}

// Streamed-input tile order.  0 (default): row-major, row i = tiles (i, 0..i) -- each
// arriving row feeds the trailing updates of every factored column at once.  1: column 0
// first (every TRSM_i_0 can start after N tiles), then the other tiles row-major.
// CHOL_ARRIVAL=0/1 (development switch, read when the plan is built).
static void arrival_order(int64_t N, int mode, std::vector<std::pair<int, int>>& tiles) {
  tiles.clear();
  if (mode == 1)
    for (int i = 0; i < N; ++i) tiles.emplace_back(i, 0);
  for (int i = 0; i < N; ++i)
    for (int j = mode == 1 ? 1 : 0; j <= i; ++j) tiles.emplace_back(i, j);
}
void sched_arrival_order(const SchedState* st, std::vector<std::pair<int, int>>& tiles) {
  arrival_order(st->N, st->arrival, tiles);
}

// Device tables of a built node graph (jobs, CSR successors, queues), the persistent grid
// size, the abort word.  Takes ownership of st (destroyed on failure).
static int sched_upload(SchedState** out, SchedState* st, Builder& B, const std::vector<int>& node_queue,
                        const std::vector<int>& publish, const std::vector<int4>& watch, const chol_opts_t* opts,
                        int64_t nb, int bs, int sms) {
  const int nnodes = (int)B.deps.size();
  if (!publish.empty() && publish.size() != (size_t)nnodes) {  // one entry per node (or none)
    sched_destroy(st);
    return -8;
  }
  // ---- queue capacities
  std::vector<int> qcap(kQueues, 0), qbase(kQueues, 0);
  for (int v = 0; v < nnodes; ++v) qcap[node_queue[v]] += 1;
  for (int q = 1; q < kQueues; ++q) qbase[q] = qbase[q - 1] + qcap[q - 1];

  std::vector<int> succ_off(nnodes + 1, 0), succ;
  for (int v = 0; v < nnodes; ++v) {
    succ_off[v + 1] = succ_off[v] + (int)B.succ[v].size();
    succ.insert(succ.end(), B.succ[v].begin(), B.succ[v].end());
  }
  std::vector<int> roots;
  for (int v = 0; v < nnodes; ++v)
    if (B.deps[v] == 0) roots.push_back(v);

  st->nnodes = nnodes;
  st->h_node_paper = B.paper;
  st->h_node_queue = node_queue;
  st->njobs = (int)B.jobs.size();
  st->h_job_type.resize(st->njobs);
  st->h_job_paper.resize(st->njobs);
  st->h_jobs = B.jobs;
  st->h_job_node = B.job_node;
  for (int j = 0; j < st->njobs; ++j) {
    st->h_job_type[j] = B.jobs[j].type;
    st->h_job_paper[j] = B.paper[B.job_node[j]];
  }
  st->nroots = (int)roots.size();

  // ---- device layout: static (read-only) part
  auto align = [](size_t x) { return (x + 255) & ~size_t(255); };
  size_t off = 0;
  const size_t o_jobs = off; off = align(off + B.jobs.size() * sizeof(Job));
  const size_t o_jnode = off; off = align(off + B.job_node.size() * 4);
  const size_t o_jbeg = off; off = align(off + nnodes * 4);
  const size_t o_jcnt = off; off = align(off + nnodes * 4);
  const size_t o_soff = off; off = align(off + (nnodes + 1) * 4);
  const size_t o_succ = off; off = align(off + std::max<size_t>(succ.size(), 1) * 4);
  const size_t o_paper = off; off = align(off + nnodes * 4);
  const size_t o_nq = off; off = align(off + nnodes * 4);
  const size_t o_qbase = off; off = align(off + kQueues * 4);
  const size_t o_roots = off; off = align(off + std::max<size_t>(roots.size(), 1) * 4);
  const size_t o_pub = off; off = align(off + (publish.empty() ? 4 : publish.size() * 4));
  const size_t o_watch = off; off = align(off + std::max<size_t>(watch.size(), 1) * 16);
  const size_t static_bytes = off;
  std::vector<char> h(static_bytes, 0);
  memcpy(h.data() + o_jobs, B.jobs.data(), B.jobs.size() * sizeof(Job));
  memcpy(h.data() + o_jnode, B.job_node.data(), B.job_node.size() * 4);
  memcpy(h.data() + o_jbeg, B.jbeg.data(), nnodes * 4);
  memcpy(h.data() + o_jcnt, B.jcnt.data(), nnodes * 4);
  memcpy(h.data() + o_soff, succ_off.data(), (nnodes + 1) * 4);
  if (!succ.empty()) memcpy(h.data() + o_succ, succ.data(), succ.size() * 4);
  memcpy(h.data() + o_paper, B.paper.data(), nnodes * 4);
  memcpy(h.data() + o_nq, node_queue.data(), nnodes * 4);
  st->o_nq = o_nq;
  st->o_qbase = o_qbase;
  memcpy(h.data() + o_qbase, qbase.data(), kQueues * 4);
  if (!roots.empty()) memcpy(h.data() + o_roots, roots.data(), roots.size() * 4);
  if (!publish.empty()) memcpy(h.data() + o_pub, publish.data(), publish.size() * 4);
  if (!watch.empty()) memcpy(h.data() + o_watch, watch.data(), watch.size() * 16);

  // dynamic part: node_deps, node_left, q_items, q_head, q_tail, done, finished
  size_t doff = 0;
  const size_t d_deps = doff; doff = align(doff + nnodes * 4);
  const size_t d_left = doff; doff = align(doff + nnodes * 4);
  const size_t pristine = doff;  // [0, pristine) is restored from the pristine copy
  const size_t d_items = doff; doff = align(doff + (size_t)nnodes * 4);
  const size_t d_next = doff; doff = align(doff + (size_t)nnodes * 4);
  const size_t d_head = doff; doff = align(doff + kQueues * kQStride * 4);
  const size_t d_tail = doff; doff = align(doff + kQueues * kQStride * 4);
  const size_t d_done = doff; doff = align(doff + 4);
  const size_t d_fin = doff; doff = align(doff + 4);
  const size_t d_fired = doff; doff = align(doff + std::max<size_t>(watch.size(), 1) * 4);
  std::vector<char> hp(pristine, 0);
  memcpy(hp.data() + d_deps, B.deps.data(), nnodes * 4);
  memcpy(hp.data() + d_left, B.jcnt.data(), nnodes * 4);

  cudaError_t e;
  if ((e = cudaMalloc(&st->dev_static, static_bytes)) || (e = cudaMalloc(&st->dev_dynamic, doff)) ||
      (e = cudaMalloc(&st->dev_pristine, pristine))) {
    cudaGetLastError();
    sched_destroy(st);
    return e == cudaErrorMemoryAllocation ? -9 : -100 - (int)e;
  }
  if ((e = cudaMemcpy(st->dev_static, h.data(), static_bytes, cudaMemcpyHostToDevice)) ||
      (e = cudaMemcpy(st->dev_pristine, hp.data(), pristine, cudaMemcpyHostToDevice))) {
    sched_destroy(st);
    return -100 - (int)e;
  }
  st->dyn_bytes = doff;
  st->pristine_bytes = pristine;
  char* S = static_cast<char*>(st->dev_static);
  char* D = static_cast<char*>(st->dev_dynamic);
  DevSched& d = st->d;
  d.jobs = reinterpret_cast<const Job*>(S + o_jobs);
  d.job_node = reinterpret_cast<const int*>(S + o_jnode);
  d.node_job_begin = reinterpret_cast<const int*>(S + o_jbeg);
  d.node_job_count = reinterpret_cast<const int*>(S + o_jcnt);
  d.succ_off = reinterpret_cast<const int*>(S + o_soff);
  d.succ = reinterpret_cast<const int*>(S + o_succ);
  d.node_paper = reinterpret_cast<const int*>(S + o_paper);
  d.node_queue = reinterpret_cast<const int*>(S + o_nq);
  d.q_base = reinterpret_cast<const int*>(S + o_qbase);
  st->roots = reinterpret_cast<int*>(S + o_roots);
  d.node_deps = reinterpret_cast<int*>(D + d_deps);
  d.node_left = reinterpret_cast<int*>(D + d_left);
  d.q_items = reinterpret_cast<int*>(D + d_items);
  d.node_next = reinterpret_cast<int*>(D + d_next);
  d.q_head = reinterpret_cast<int*>(D + d_head);
  d.q_tail = reinterpret_cast<int*>(D + d_tail);
  d.done_nodes = reinterpret_cast<int*>(D + d_done);
  d.finished = reinterpret_cast<int*>(D + d_fin);
  d.total_nodes = nnodes;
  d.node_publish = publish.empty() ? nullptr : reinterpret_cast<const int*>(S + o_pub);
  d.watch = reinterpret_cast<const int4*>(S + o_watch);
  d.nwatch = (int)watch.size();
  d.watch_fired = reinterpret_cast<int*>(D + d_fired);
  d.nb = (int)nb;
  st->nrecv_jobs = 0;
  for (const Job& jb : B.jobs) st->nrecv_jobs += jb.type == J_RECV;
  if (opts->trace == 2) {
    if ((e = cudaMalloc(&st->job_trace, (size_t)st->njobs * 4 * sizeof(uint64_t)))) {
      cudaGetLastError();
      sched_destroy(st);
      return -9;
    }
  }
  d.job_trace = st->job_trace;
  d.policy = opts->policy;
  d.latency_workers = opts->policy == CHOL_POLICY_STATIC ? (opts->latency_workers > 0 ? opts->latency_workers : 16) : 0;

  // ---- workers: one CTA per SM (all co-resident)
  int per_sm = 0;
  const int smem = smem_bytes(bs);
  cudaError_t ea = cudaSuccess;
  switch (bs) {
    case 96: ea = cudaFuncSetAttribute(k_sched<96>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
             if (!ea) ea = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_sched<96>, kWsThreads, smem); break;
    case 64: ea = cudaFuncSetAttribute(k_sched<64>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
             if (!ea) ea = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_sched<64>, kWsThreads, smem); break;
    case 32: ea = cudaFuncSetAttribute(k_sched<32>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
             if (!ea) ea = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_sched<32>, kWsThreads, smem); break;
  }
  if (ea || per_sm < 1) {
    sched_destroy(st);
    return ea ? -100 - (int)ea : -8;
  }
  st->workers = opts->workers > 0 ? std::min(opts->workers, sms * per_sm) : sms;
  if (d.latency_workers >= st->workers) d.latency_workers = std::max(1, st->workers / 4);

  {
    // device memory, not host-mapped: the scheduler warps read it whenever they idle
    cudaError_t ea = cudaMalloc(&st->d_abort, sizeof(int));
    if (!ea) ea = cudaMemset(st->d_abort, 0, sizeof(int));
    if (ea) {
      sched_destroy(st);
      return -100 - (int)ea;
    }
    st->d.abort_flag = st->d_abort;
  }
    *out = st;
  return 0;
}

int sched_create(SchedState** out, int64_t N, int64_t nb, int bs, int sms, const chol_opts_t* opts,
                 cudaStream_t /*s*/, const DistInfo* dist) {
  auto* st = new SchedState();
  const char* ear = getenv("CHOL_ARRIVAL");
  st->arrival = ear ? atoi(ear) : 0;
  st->N = N;
  st->nb = nb;
  st->bs = bs;
  st->opts = *opts;
  const int nbb = (int)(nb / bs);
  Builder B{N, nbb, opts->policy, opts->trsm_pin_distance > 0 ? opts->trsm_pin_distance : 1};

  // TRSM decomposition: row-slab jobs (default) or right-looking block nodes
  // (CHOL_TRSM_BLOCKS=1, development switch; measured 2.5% slower at n=19200).
  const char* ev = getenv("CHOL_TRSM_BLOCKS");
  const bool trsm_slab_all = !(ev && ev[0] == '1');
  // Steps whose TRSMs are on the critical path use the block decomposition (TS/TU:
  // more parallel, ~2.5x shorter latency than a 500 us slab job): the last step always,
  // every step of a small factorization (N <= 8).  Measured (job traces, r01): n=19200
  // 72.02 -> 71.79 ms, n=3840 4.40 -> 4.04 ms, n=1920 1.84 -> 1.72 ms.
  // CHOL_TRSM_TAIL=t overrides (last t steps; development switch).
  const char* et = getenv("CHOL_TRSM_TAIL");
  const int trsm_tail = et ? atoi(et) : (N <= 8 ? (int)N : 1);
  // ... and the TRSMs within trsm_dist tiles of the diagonal at every step (TRSM_{k+1,k}
  // is on the chain POTRF_k -> TRSM_{k+1,k} -> SYRK_{k+1,k} -> POTRF_{k+1}).
  // CHOL_TRSM_DIST=d overrides (development switch).
  const char* etd = getenv("CHOL_TRSM_DIST");
  const int trsm_dist = etd ? atoi(etd) : 0;
  // TS/TU decomposition: per-column-step nodes (0, default) or per-row-slab chains of
  // single-job nodes (1; measured slower under load).  CHOL_TRSM_SLABCHAIN.
  const char* esc = getenv("CHOL_TRSM_SLABCHAIN");
  const bool trsm_slabchain = esc && atoi(esc) != 0;
  // POTRF inner structure: block-level DAG (one job per node: the chain D -> P -> U -> D
  // never waits for a whole inner step) or per-step nodes (DIAG b, PANEL b, UPDATE b:
  // 28 nodes per POTRF instead of 220).  The block DAG shortens the POTRF chain
  // (785 -> 633 us alone, n=9600 15.1 -> 13.3 ms) but its extra nodes cost dispatch
  // work: 0.3 ms at n=19200, where the area bound dominates (chain/area ~ 141/N^2 at
  // nb=960).  Default: block DAG while N <= 16, i.e. N^2 <= 256 tiles per GPU -- a rank
  // of an R-GPU plan holds ~N^2/R of the area but the whole chain, so the same rule
  // reads N^2 / R <= 256 there.  CHOL_POTRF_BLOCKDAG=0/1 overrides.
  const char* epb = getenv("CHOL_POTRF_BLOCKDAG");
  const int64_t ranks = dist ? std::max(1, dist->nranks) : 1;
  const bool potrf_blockdag = epb ? atoi(epb) != 0 : N * N <= 256 * ranks;
  // POTRF block DAG: the diagonal block's last update fused into its potf2 job
  // (CHOL_POTRF_FUSE=0 turns it off; development switch)
  const char* epf = getenv("CHOL_POTRF_FUSE");
  const bool potrf_fuse = !(epf && atoi(epf) == 0);
  const char* ep0 = getenv("CHOL_POTRF0_BLOCKDAG");
  const bool potrf0_blockdag = !(ep0 && atoi(ep0) == 0);
  // Hybrid DAG: the steps k >= k0 are built at BS-block granularity across tasks (the
  // paper's tasks keep their kernels, but a consumer block waits only for the producer
  // blocks it reads): POTRF as its block DAG, TRSM as per-slab chains (TS/TU), SYRK and
  // GEMM as one node per BS x BS output block (K = nb), with block-level edges between
  // them.  Where the run is chain-bound (small N, the last steps of any N) the next
  // step's POTRF then starts as soon as its first blocks are updated instead of after
  // the whole SYRK.  A larger block region costs efficiency (K = BS TRSM updates, more
  // nodes): measured best m (tools/tail_sweep.py, nb = 960) is 4 for N = 4..10 and 2 for
  // N = 12..24 (n=3840 3.76 -> 2.82 ms, n=9600 13.07 -> 12.18, n=19200 71.82 -> 71.57).
  // Distributed plans too (round 2): a remote panel tile enters the blocked region through
  // its RECV node, which every block node reading it waits for.  CHOL_BLOCK_TAIL=m overrides
  // (m steps).
  const char* ebt = getenv("CHOL_BLOCK_TAIL");
  // round-2 sweep (profiles/r02/block_tail_sweep_r02.txt): m = 4 for N <= 6, 3 for N = 7..10
  // (n=9600 11.78 -> 11.25 ms, n=7680 8.11 -> 7.93), 2 above
  int block_tail = ebt ? atoi(ebt) : (N <= 6 ? 4 : N <= 10 ? 3 : 2);
  const int k0 = (int)N - std::max(0, std::min(block_tail, (int)N));
  // blocked-region TRSM: per-slab TS/TU chains (0) or one left-looking slab job per
  // slab node (1).  CHOL_TAIL_TRSM.
  const char* ett = getenv("CHOL_TAIL_TRSM");
  const bool tail_trsm_slab = ett && atoi(ett) == 1;
  // Multi-GPU: this rank creates the nodes of the tasks that overwrite the tiles it owns
  // (owner-computes), plus one RECV node per remote panel tile it reads.
  auto mine = [&](int64_t i, int64_t j) { return !dist || tile_owner(i, j, dist->p, dist->q) == dist->rank; };
  std::vector<int> publish;  // per node: tile made final (published to other ranks) or -1
  // ---- nodes and jobs, Algorithm 1 order
  std::vector<int> first_node(n_tasks(N), -1), last_node(n_tasks(N), -1);
  // blocked tasks (k >= k0): per BS x BS block of the tile the task writes, the node that
  // first touches it (tentry) and the node that leaves it final (tfin); TRSM: the node
  // that finishes each row slab (tslab)
  std::vector<std::vector<int>> tentry(n_tasks(N)), tfin(n_tasks(N)), tslab(n_tasks(N));
  // inverse-form TRSM row slabs of each step and the D(b) nodes of each local POTRF
  // (build_inverses, after the task edges)
  std::vector<std::vector<int>> slab_nodes(N), dnodes(N);
  // host CPU class: TRSMs at least cpu_d tiles below the diagonal (0 = off; single GPU)
  const int cpu_d = dist ? 0 : opts->cpu_trsm_distance;
  std::vector<int> host_in, host_out;
  std::vector<std::vector<std::vector<int>>> ts_nodes(N, std::vector<std::vector<int>>(nbb));
  const int nbb2 = nbb * nbb;
  std::vector<int4> watch;  // multi-GPU: {RECV node, owner, tile, step}
  std::vector<int> recv_node((size_t)(N * (N + 1) / 2), -1);  // multi-GPU: RECV node of a remote tile
  // multi-GPU: this rank's RECV node for remote panel tile (i, j), created on first use (its
  // jobs copy the tile's row slabs from the owner's store; the watcher fires it when the
  // owner publishes the tile)
  auto recv_of = [&](int64_t i, int64_t j) -> int {
    const int64_t t = tile_index(i, j);
    if (recv_node[t] < 0) {
      const int owner = tile_owner((int)i, (int)j, dist->p, dist->q);
      const int rn = B.add_node(-1, -1, (int)i, (int)j);
      for (int sl = 0; sl < nbb; ++sl)
        B.add_job(rn, Job{J_RECV, (int16_t)i, (int16_t)j, 0, (int16_t)sl, (int16_t)owner, 0, 0});
      B.deps[rn] += 1;  // fired by the watcher (remote readiness)
      recv_node[t] = rn;
      watch.push_back(make_int4(rn, owner, (int)t, (int)j));
    }
    return recv_node[t];
  };
  // the node that makes block (r, c) of L_kk final: local D / P node, or the RECV of L_kk
  auto lkk_block = [&](int k, int pid, int r, int c) { return mine(k, k) ? tfin[pid][r * nbb + c] : recv_of(k, k); };
  auto gate_of = [&](int tid, int type, int i, int k) {
    // job-less node in front of a blocked task's entry nodes: the target of task-level
    // dependencies (streamed tile arrival at k = 0)
    const int gate = B.add_node(tid, type, i, k);
    std::vector<int> seen;
    for (int e : tentry[tid])
      if (e >= 0 && std::find(seen.begin(), seen.end(), e) == seen.end()) {
        B.edge(gate, e);
        seen.push_back(e);
      }
    first_node[tid] = gate;
  };
  for (int k = 0; k < N; ++k) {
    const int pid = (int)id_potrf(N, k);
    const bool blk = k >= k0;
    // POTRF_0 runs alone on an idle GPU (every other task depends on it): always the
    // shorter block DAG (CHOL_POTRF0_BLOCKDAG=0 turns this off; development switch)
    const bool pblock = potrf_blockdag || (k == 0 && potrf0_blockdag);
    if (mine(k, k) && !pblock && !blk) {  // per-step nodes: DIAG b -> PANEL b -> UPDATE b
      build_potrf_steps(B, k, pid, &first_node[pid], &last_node[pid], &dnodes[k]);
    } else if (mine(k, k)) {
      build_potrf_blockdag(B, k, pid, potrf_fuse, blk, &tentry[pid], &tfin[pid], &first_node[pid], &last_node[pid],
                           &dnodes[k]);
      if (blk && k == 0) gate_of(pid, T_POTRF, k, k);
    }
    for (int i = k + 1; i < N && blk; ++i) {
      // blocked TRSM_i_k: per row slab sl, TS(c, sl) / TU(c, sl, c') single-job nodes
      // (or one slab job per node), edges from the POTRF_k blocks each one reads:
      // TS(c, sl) <- L_kk[c,c] = D(c); TU(c, sl, c') <- L_kk[c',c] = P(c',c)
      if (!mine(i, k)) continue;
      const int tid = (int)id_trsm(N, i, k);
      tentry[tid].assign(nbb2, -1);
      tfin[tid].assign(nbb2, -1);
      tslab[tid].assign(nbb, -1);
      const int exit_ = B.add_node(tid, T_TRSM, i, k);  // job-less: the tile is final (publish)
      for (int sl = 0; sl < nbb; ++sl) {
        if (tail_trsm_slab) {
          const int sn = B.add_node(tid, T_TRSM, i, k);
          B.add_job(sn, Job{J_TRSM, (int16_t)i, (int16_t)k, (int16_t)k, (int16_t)sl, 0, 0, 0});
          B.edge(lkk_block(k, pid, nbb - 1, nbb - 1), sn);  // D(nbb-1): all of L_kk
          slab_nodes[k].push_back(sn);
          for (int c = 0; c < nbb; ++c) tentry[tid][sl * nbb + c] = tfin[tid][sl * nbb + c] = sn;
          tslab[tid][sl] = sn;
          B.edge(sn, exit_);
          continue;
        }
        std::vector<int> lastTU(nbb, -1);
        for (int cb = 0; cb < nbb; ++cb) {
          const int ts = B.add_node(tid, T_TRSM, i, k);
          B.add_job(ts, Job{J_TS, (int16_t)i, (int16_t)k, (int16_t)k, (int16_t)cb, (int16_t)sl, 0, 0});
          ts_nodes[k][cb].push_back(ts);
          B.edge(lkk_block(k, pid, cb, cb), ts);
          if (cb > 0) B.edge(lastTU[cb], ts);
          else tentry[tid][sl * nbb] = ts;
          tfin[tid][sl * nbb + cb] = ts;
          for (int c2 = cb + 1; c2 < nbb; ++c2) {
            const int tu = B.add_node(tid, T_TRSM, i, k);
            B.add_job(tu, Job{J_TU, (int16_t)i, (int16_t)k, (int16_t)k, (int16_t)cb, (int16_t)sl, (int16_t)c2, 0});
            B.edge(ts, tu);
            B.edge(lkk_block(k, pid, c2, cb), tu);
            if (lastTU[c2] >= 0) B.edge(lastTU[c2], tu);
            else tentry[tid][sl * nbb + c2] = tu;
            lastTU[c2] = tu;
          }
        }
        tslab[tid][sl] = tfin[tid][sl * nbb + nbb - 1];
        B.edge(tslab[tid][sl], exit_);
      }
      last_node[tid] = exit_;
      if (k == 0) gate_of(tid, T_TRSM, i, k);
    }
    for (int i = k + 1; i < N && !blk; ++i) {
      if (!mine(i, k)) continue;
      if (cpu_d > 0 && i - k >= cpu_d) {
        // host CPU class (NEXT-3, the paper's TRSM-distance rule, L1019-1025): OUT (one no-op
        // job) publishes "inputs final" to the host; IN (job-less) is fired by the watcher when
        // the host has written L_ik back; IN is the task's last node (publishes the tile)
        const int tid = (int)id_trsm(N, i, k);
        const int outn = B.add_node(tid, T_TRSM, i, k);
        B.add_job(outn, Job{J_NOP, (int16_t)i, (int16_t)k, (int16_t)k, 0, 0, 0, 0});
        const int inn = B.add_node(-1, T_TRSM, i, k);
        host_in.push_back(inn);
        host_out.push_back(outn);
        st->host_tasks.emplace_back(i, k);
        first_node[tid] = outn;
        last_node[tid] = inn;
        slab_nodes[k].push_back(outn);  // waits for the inverses Dinv_k too
        continue;
      }
      const bool trsm_slab = trsm_slab_all && k < N - 1 - trsm_tail && i - k > trsm_dist;
      if (trsm_slab) {  // one left-looking row-slab job per BS rows
        const int tid = (int)id_trsm(N, i, k);
        const int n = B.add_node(tid, T_TRSM, i, k);
        for (int sl = 0; sl < nbb; ++sl)
          B.add_job(n, Job{J_TRSM, (int16_t)i, (int16_t)k, (int16_t)k, (int16_t)sl, 0, 0, 0});
        first_node[tid] = last_node[tid] = n;
        slab_nodes[k].push_back(n);
        continue;
      }
      if (!trsm_slabchain) {  // right-looking column steps TS(c) / TU(c)
        const int tid = (int)id_trsm(N, i, k);
        build_trsm_steps(B, i, k, tid, &first_node[tid], &last_node[tid], &ts_nodes[k]);
        continue;
      }
      // Alternative (CHOL_TRSM_SLABCHAIN=1): rows are independent (X L^{-T}), so each
      // BS-row slab sl is its own chain:
      //   TS(c, sl): A_ik[sl, c] <- A_ik[sl, c] L_kk[c,c]^{-T}
      //   TU(c, sl, c'): A_ik[sl, c'] -= A_ik[sl, c] L_kk[c',c]^T, c' > c   (K = BS)
      // one job per node; a job-less entry node fans out to the nbb chains and a
      // job-less exit node joins them (the task's single first / last node).
      const int tid = (int)id_trsm(N, i, k);
      const int entry = B.add_node(tid, T_TRSM, i, k), exit_ = B.add_node(tid, T_TRSM, i, k);
      first_node[tid] = entry;
      last_node[tid] = exit_;
      std::vector<int> lastTU(nbb, -1);
      for (int sl = 0; sl < nbb; ++sl) {
        std::fill(lastTU.begin(), lastTU.end(), -1);
        for (int cb = 0; cb < nbb; ++cb) {
          const int ts = B.add_node(tid, T_TRSM, i, k);
          B.add_job(ts, Job{J_TS, (int16_t)i, (int16_t)k, (int16_t)k, (int16_t)cb, (int16_t)sl, 0, 0});
          ts_nodes[k][cb].push_back(ts);
          B.edge(cb == 0 ? entry : lastTU[cb], ts);
          if (cb + 1 == nbb) B.edge(ts, exit_);
          for (int c2 = cb + 1; c2 < nbb; ++c2) {
            const int tu = B.add_node(tid, T_TRSM, i, k);
            B.add_job(tu, Job{J_TU, (int16_t)i, (int16_t)k, (int16_t)k, (int16_t)cb, (int16_t)sl, (int16_t)c2, 0});
            B.edge(ts, tu);
            if (lastTU[c2] >= 0) B.edge(lastTU[c2], tu);
            lastTU[c2] = tu;
          }
        }
      }
    }
    for (int j = k + 1; j < N && blk; ++j) {
      // blocked SYRK_j_k / GEMM_i_j_k: one node per output block, K = nb
      const int sid = (int)id_syrk(N, j, k);
      if (mine(j, j)) {
        tentry[sid].assign(nbb2, -1);
        for (int bm = 0; bm < nbb; ++bm)
          for (int bn = 0; bn <= bm; ++bn) {
            const int n = B.add_node(sid, T_SYRK, j, k);
            B.add_job(n, Job{J_UPD, (int16_t)j, (int16_t)j, (int16_t)k, (int16_t)bm, (int16_t)bn, 0, 0});
            tentry[sid][bm * nbb + bn] = n;
          }
        tfin[sid] = tentry[sid];
        if (k == 0) gate_of(sid, T_SYRK, j, k);
      }

      for (int i = j + 1; i < N; ++i) {
        if (!mine(i, j)) continue;
        const int gid = (int)id_gemm(N, i, j, k);
        tentry[gid].assign(nbb2, -1);
        for (int bm = 0; bm < nbb; ++bm)
          for (int bn = 0; bn < nbb; ++bn) {
            const int g = B.add_node(gid, T_GEMM, i, k);
            B.add_job(g, Job{J_UPD, (int16_t)i, (int16_t)j, (int16_t)k, (int16_t)bm, (int16_t)bn, 0, 0});
            tentry[gid][bm * nbb + bn] = g;
          }
        tfin[gid] = tentry[gid];
        if (k == 0) gate_of(gid, T_GEMM, i, k);
      }
    }
    for (int j = k + 1; j < N && !blk; ++j) {
      const int sid = (int)id_syrk(N, j, k);
      if (mine(j, j)) {
        const int n = B.add_node(sid, T_SYRK, j, k);
        for (int bm = 0; bm < nbb; ++bm)
          for (int bn = 0; bn <= bm; ++bn)
            B.add_job(n, Job{J_UPD, (int16_t)j, (int16_t)j, (int16_t)k, (int16_t)bm, (int16_t)bn, 0, 0});
        first_node[sid] = last_node[sid] = n;
      }
      for (int i = j + 1; i < N; ++i) {
        if (!mine(i, j)) continue;
        const int gid = (int)id_gemm(N, i, j, k);
        const int g = B.add_node(gid, T_GEMM, i, k);
        for (int bm = 0; bm < nbb; ++bm)
          for (int bn = 0; bn < nbb; ++bn)
            B.add_job(g, Job{J_UPD, (int16_t)i, (int16_t)j, (int16_t)k, (int16_t)bm, (int16_t)bn, 0, 0});
        first_node[gid] = last_node[gid] = g;
      }
    }
  }

  // ---- task edges: direct data dependencies of Algorithm 1 (dag.cpp, L213-220),
  // mapped onto the nodes (POTRF_k enters at its first inner node, leaves at its last).
  std::vector<std::pair<int64_t, int64_t>> E;
  std::vector<int> type_of;
  build_task_dag(N, E, type_of);
  // tile written by a task (i, j) -- Algorithm 1 visit order of taskid.h
  std::vector<int2> wtile(n_tasks(N));
  for (int64_t k = 0; k < N; ++k) {
    wtile[id_potrf(N, k)] = make_int2((int)k, (int)k);
    for (int64_t i = k + 1; i < N; ++i) wtile[id_trsm(N, i, k)] = make_int2((int)i, (int)k);
    for (int64_t j = k + 1; j < N; ++j) {
      wtile[id_syrk(N, j, k)] = make_int2((int)j, (int)j);
      for (int64_t i = j + 1; i < N; ++i) wtile[id_gemm(N, i, j, k)] = make_int2((int)i, (int)j);
    }
  }
  // Multi-GPU: a rank builds the edges into the tasks it owns; a producer on another rank
  // (always the task that made a panel tile L_kk / L_ik final) is reached through this
  // rank's RECV node for that tile, which every node of the consumer waits for.
  auto owned = [&](int64_t task) { return mine(wtile[task].x, wtile[task].y); };
  for (auto& e : E) {
    const int64_t a = e.first, b = e.second;
    if (dist && !owned(b)) continue;
    if (dist && !owned(a)) {
      const int rn = recv_of(wtile[a].x, wtile[a].y);
      if (tentry[b].empty()) {
        B.edge(rn, first_node[b]);
      } else if (!(type_of[a] == T_POTRF && type_of[b] == T_TRSM)) {  // TRSM blocks: made with the nodes
        std::vector<int> seen;
        for (int x : tentry[b])
          if (x >= 0 && std::find(seen.begin(), seen.end(), x) == seen.end()) {
            B.edge(rn, x);
            seen.push_back(x);
          }
      }
      continue;
    }
    if (tentry[b].empty()) {  // task-level consumer (k < k0)
      B.edge(last_node[a], first_node[b]);
      continue;
    }
    const int2 tb = wtile[b];
    const bool diag = tb.x == tb.y;
    if (tentry[a].empty()) {  // task-level producer of a blocked consumer: every entry waits
      std::vector<int> seen;
      for (int x : tentry[b])
        if (x >= 0 && std::find(seen.begin(), seen.end(), x) == seen.end()) {
          B.edge(last_node[a], x);
          seen.push_back(x);
        }
      continue;
    }
    if (type_of[a] == T_POTRF && type_of[b] == T_TRSM) continue;  // block edges made with the TRSM nodes
    for (int bm = 0; bm < nbb; ++bm)
      for (int bn = 0; bn < nbb; ++bn) {
        if (diag && bn > bm) continue;  // lower blocks of a diagonal tile
        const int x = tentry[b][bm * nbb + bn];
        if (x < 0) continue;
        if (type_of[a] == T_TRSM) {  // L_ik read by SYRK / GEMM: row slabs bm and / or bn
          const int pi = wtile[a].x;
          if (pi == tb.x) B.edge(tslab[a][bm], x);
          if (pi == tb.y && !(pi == tb.x && bm == bn)) B.edge(tslab[a][bn], x);
        } else {  // the same tile, block by block (SYRK->POTRF, SYRK->SYRK, GEMM->GEMM, GEMM->TRSM)
          B.edge(tfin[a][bm * nbb + bn], x);
        }
      }
  }
  if (!dist) {
    // Streamed input (chol_factor from host memory): the first task touching a tile
    // waits for the tile's arrival flag (the copy engine writes it after the tile).
    // Tiles arrive in row-major tile order (row i: tiles (i,0..i)); the watch list
    // follows the same order.  Row-major arrival lets each arriving row feed the
    // trailing updates of every factored column at once (list-scheduling model of
    // the job DAG, 148 workers, 53.6 GB/s: 72.2 ms vs 73.8 ms for column order and
    // 70.6 ms for instant arrival at n=19200).
    int order = 0;
    auto first_touch = [&](int64_t task, int64_t i, int64_t j) {
      const int64_t t = tile_index(i, j);
      B.deps[first_node[task]] += 1;
      watch.push_back(make_int4(first_node[task], 0, (int)t, order++));
    };
    std::vector<std::pair<int, int>> arr;
    arrival_order(N, st->arrival, arr);
    for (const auto& ij : arr) {
      const int64_t i = ij.first, j = ij.second;
      if (j == 0)
        first_touch(i == 0 ? id_potrf(N, 0) : id_trsm(N, i, 0), i, 0);  // POTRF_0 / TRSM_i_0
      else if (i == j)
        first_touch(id_syrk(N, j, 0), j, j);  // SYRK_j_0
      else
        first_touch(id_gemm(N, i, j, 0), i, j);  // GEMM_i_j_0
    }
    // Streamed output: every final panel tile is published (host-mapped flags)
    publish.assign(B.deps.size(), -1);
    for (int64_t k = 0; k < N; ++k) {
      publish[last_node[id_potrf(N, k)]] = (int)tile_index(k, k);
      for (int64_t i = k + 1; i < N; ++i) publish[last_node[id_trsm(N, i, k)]] = (int)tile_index(i, k);
    }
    // host CPU class: OUT publishes into the second half of the host-mapped flag array
    // ("inputs of tile t final"); IN waits for the host's flag (peer_flags[1], watch order
    // after every input-arrival entry)
    const int64_t ntl = N * (N + 1) / 2;
    for (size_t h = 0; h < host_in.size(); ++h) {
      const int i = st->host_tasks[h].first, k = st->host_tasks[h].second;
      const int t = (int)tile_index(i, k);
      publish[host_out[h]] = (int)(ntl + t);
      B.deps[host_in[h]] += 1;
      watch.push_back(make_int4(host_in[h], 1, t, (int)(ntl + h)));
    }
  } else {
    std::stable_sort(watch.begin(), watch.end(), [](const int4& a, const int4& b) { return a.w < b.w; });
    // panel tiles this rank finalises are published (their final node)
    publish.assign(B.deps.size(), -1);
    for (int64_t k = 0; k < N; ++k) {
      if (mine(k, k)) publish[last_node[id_potrf(N, k)]] = (int)tile_index(k, k);
      for (int64_t i = k + 1; i < N; ++i)
        if (mine(i, k)) publish[last_node[id_trsm(N, i, k)]] = (int)tile_index(i, k);
    }
  }

  // ---- inverses of the diagonal blocks of L_kk for the inverse-form TRSM row slabs: after
  // the local D(b) nodes, or after the RECV of a remote L_kk
  for (int k = 0; k < N; ++k) {
    std::vector<int> pred = dnodes[k];
    if (pred.empty() && recv_node[tile_index(k, k)] >= 0) pred.assign(1, recv_node[tile_index(k, k)]);
    build_inverses(B, k, pred, slab_nodes[k], ts_nodes[k]);
  }
  if (!publish.empty()) publish.resize(B.deps.size(), -1);  // the inverse nodes publish nothing

  // ---- priorities: bottom-level of each Algorithm 1 task (HEFT / dmdas, L299-301,
  // L655-660; reading R13) with latency-estimate weights, quantised into kBuckets;
  // POTRF's inner nodes inherit the POTRF priority.
  const int nnodes = (int)B.deps.size();
  double w_type[4] = {300.0, 300.0, 80.0, 80.0};
  if (const char* ew = getenv("CHOL_PRIO_W"))  // development switch: "p,t,s,g" (us)
    sscanf(ew, "%lf,%lf,%lf,%lf", &w_type[0], &w_type[1], &w_type[2], &w_type[3]);
  const std::vector<double> bl = bottom_levels(N, w_type);
  const double blmax = *std::max_element(bl.begin(), bl.end()) + 1e-9;
  std::vector<int> node_queue(nnodes, 0);
  for (int v = 0; v < nnodes; ++v) {
    int bucket = 0;
    if (opts->policy != CHOL_POLICY_DYNAMIC)
      bucket = B.paper[v] < 0 ? kBuckets - 1  // RECV: gates local work
                              : std::min(kBuckets - 1, (int)(kBuckets * bl[B.paper[v]] / blmax));
    bool pinned = false;
    if (opts->policy == CHOL_POLICY_STATIC) {
      if (B.ptype[v] == T_POTRF) pinned = true;
      if (B.ptype[v] == T_TRSM && B.pi[v] - B.pk[v] <= B.pin_d) pinned = true;
    }
    node_queue[v] = bucket + (pinned ? kBuckets : 0);
  }

  return sched_upload(out, st, B, node_queue, publish, watch, opts, nb, bs, sms);
}

// Calibration batches (chol_run_batch; reading R9): `count` independent tasks of
// one type on distinct output tiles, no edges -- POTRF on diagonal tiles 0..count-1,
// TRSM_{i,k} over the N(N-1)/2 panel tiles in Algorithm 1 order (k, then i: enough
// instances to saturate the GPU with row-slab jobs), SYRK_{c+1,0}, GEMM_{i,j,0} over the
// pairs N > i > j >= 1 (j ascending, then i) -- run by the same persistent kernel as the factorization and in the
// same job decompositions: the bulk forms when count > 1 (row-slab TRSM jobs; per-step POTRF
// nodes wherever the factorization uses them), the critical-path forms when count == 1
// (right-looking TRSM column steps, the POTRF block DAG).
int sched_create_batch(SchedState** out, int64_t N, int64_t nb, int bs, int sms, const chol_opts_t* opts, int type,
                       int count) {
  const int maxc = type == T_POTRF   ? (int)N
                   : type == T_GEMM  ? (int)((N - 1) * (N - 2) / 2)
                   : type == T_TRSM  ? (int)(N * (N - 1) / 2)
                                     : (int)N - 1;
  if (type < 0 || type > 3 || count < 1 || count > maxc) return -6;
  auto* st = new SchedState();
  st->N = N;
  st->nb = nb;
  st->bs = bs;
  st->opts = *opts;
  const int nbb = (int)(nb / bs);
  Builder B{N, nbb, opts->policy, 1};
  const char* epb = getenv("CHOL_POTRF_BLOCKDAG");
  const bool potrf_blockdag = count == 1 || (epb ? atoi(epb) != 0 : N * N <= 256);
  const char* epf = getenv("CHOL_POTRF_FUSE");
  const bool potrf_fuse = !(epf && atoi(epf) == 0);
  int first = -1, last = -1, c = 0;
  if (type == T_POTRF) {
    for (int k = 0; k < count; ++k) {
      if (potrf_blockdag)
        build_potrf_blockdag(B, k, -1, potrf_fuse, false, nullptr, nullptr, &first, &last);
      else
        build_potrf_steps(B, k, -1, &first, &last);
    }
  } else if (type == T_TRSM) {
    std::vector<std::vector<int>> slabs(N);
    for (int k = 0; k < N && c < count; ++k)
      for (int i = k + 1; i < N && c < count; ++i, ++c) {
        if (count == 1) {
          std::vector<std::vector<int>> ts;
          build_trsm_steps(B, i, k, -1, &first, &last, &ts);
          build_inverses(B, k, {}, {}, ts);
          continue;
        }
        const int n = B.add_node(-1, T_TRSM, i, k);
        for (int sl = 0; sl < nbb; ++sl)
          B.add_job(n, Job{J_TRSM, (int16_t)i, (int16_t)k, (int16_t)k, (int16_t)sl, 0, 0, 0});
        slabs[k].push_back(n);
      }
    for (int k = 0; k < N; ++k) build_inverses(B, k, {}, slabs[k]);  // part of the TRSM cost
  } else if (type == T_SYRK) {
    for (int j = 1; j <= count; ++j) {
      const int n = B.add_node(-1, T_SYRK, j, 0);
      for (int bm = 0; bm < nbb; ++bm)
        for (int bn = 0; bn <= bm; ++bn)
          B.add_job(n, Job{J_UPD, (int16_t)j, (int16_t)j, 0, (int16_t)bm, (int16_t)bn, 0, 0});
    }
  } else {
    for (int j = 1; j < N && c < count; ++j)
      for (int i = j + 1; i < N && c < count; ++i, ++c) {
        const int g = B.add_node(-1, T_GEMM, i, 0);
        for (int bm = 0; bm < nbb; ++bm)
          for (int bn = 0; bn < nbb; ++bn)
            B.add_job(g, Job{J_UPD, (int16_t)i, (int16_t)j, 0, (int16_t)bm, (int16_t)bn, 0, 0});
      }
  }
  std::vector<int> node_queue(B.deps.size(), 0), publish;
  std::vector<int4> watch;
  return sched_upload(out, st, B, node_queue, publish, watch, opts, nb, bs, sms);
}

// Injected static priorities (NEXT-4: the paper injects its CP schedules into StarPU,
// P:L1063-1072): prio[paper task id] (higher = earlier) replaces the bottom-level bucket of
// every task node; pinned classes (STATIC) and the untraced gating nodes (RECV, INV: top
// bucket) are kept.  Rewrites the node -> queue table and the queue bases on the device.
int sched_set_priorities(SchedState* st, const double* prio, int64_t ntasks) {
  if (!st || !prio) return -4;
  if (ntasks != n_tasks(st->N)) return -6;
  double lo = prio[0], hi = prio[0];
  for (int64_t t = 1; t < ntasks; ++t) lo = std::min(lo, prio[t]), hi = std::max(hi, prio[t]);
  const double span = hi - lo > 0 ? hi - lo : 1.0;
  std::vector<int> nq(st->nnodes);
  for (int v = 0; v < st->nnodes; ++v) {
    const int pinned = st->h_node_queue[v] >= kBuckets ? kBuckets : 0;
    const int p = st->h_node_paper[v];
    const int bucket = p < 0 ? kBuckets - 1 : std::min(kBuckets - 1, (int)((kBuckets - 1) * (prio[p] - lo) / span));
    nq[v] = bucket + pinned;
  }
  std::vector<int> qcap(kQueues, 0), qbase(kQueues, 0);
  for (int v = 0; v < st->nnodes; ++v) qcap[nq[v]] += 1;
  for (int q = 1; q < kQueues; ++q) qbase[q] = qbase[q - 1] + qcap[q - 1];
  char* S = static_cast<char*>(st->dev_static);
  cudaError_t e = cudaMemcpy(S + st->o_nq, nq.data(), nq.size() * 4, cudaMemcpyHostToDevice);
  if (!e) e = cudaMemcpy(S + st->o_qbase, qbase.data(), kQueues * 4, cudaMemcpyHostToDevice);
  if (e) return -100 - (int)e;
  st->h_node_queue = nq;
  return 0;
}

int sched_set_dinv(SchedState* st, double* dinv, const CUtensorMap& dmap) {
  st->d.dinv = dinv;
  st->dmap = dmap;
  return 0;
}

int sched_set_dist(SchedState* st, const int* d_slot_map, const int* d_owner_slot, double* const* d_peer_slots,
                   int* const* d_peer_flags, int* d_my_flags) {
  st->d.slot_map = d_slot_map;
  st->d.owner_slot = d_owner_slot;
  st->d.peer_slots = d_peer_slots;
  st->d.peer_flags = d_peer_flags;
  st->d.my_flags = d_my_flags;
  return 0;
}

int sched_run(SchedState* st, const CUtensorMap& map, const StepParams& base, cudaStream_t s, int* nlaunch,
              unsigned epoch) {
  st->d.epoch = epoch;
  cudaError_t e;
  if ((e = cudaMemsetAsync(st->d_abort, 0, sizeof(int), s))) return -100 - (int)e;
  if ((e = cudaMemcpyAsync(st->dev_dynamic, st->dev_pristine, st->pristine_bytes, cudaMemcpyDeviceToDevice, s)))
    return -100 - (int)e;
  if ((e = cudaMemsetAsync(static_cast<char*>(st->dev_dynamic) + st->pristine_bytes, 0,
                           st->dyn_bytes - st->pristine_bytes, s)))
    return -100 - (int)e;
  st->d.tr_base = base.tr_base;
  if (!base.tr_base) st->d.job_trace = nullptr;  // job trace needs the time base
  else st->d.job_trace = st->job_trace;
  k_sched_init<<<std::max(1, std::min(64, (st->nroots + 127) / 128)), 128, 0, s>>>(st->d, st->roots, st->nroots);
  const int smem = smem_bytes(st->bs);
  switch (st->bs) {
    case 96: k_sched<96><<<st->workers, kWsThreads, smem, s>>>(map, st->dmap, base, st->d); break;
    case 64: k_sched<64><<<st->workers, kWsThreads, smem, s>>>(map, st->dmap, base, st->d); break;
    case 32: k_sched<32><<<st->workers, kWsThreads, smem, s>>>(map, st->dmap, base, st->d); break;
  }
  *nlaunch += 2;
  if ((e = cudaGetLastError())) return -100 - (int)e;
  return 0;
}

int sched_workers(const SchedState* st) { return st ? st->workers : 0; }
const std::vector<std::pair<int, int>>& sched_host_tasks(const SchedState* st) { return st->host_tasks; }
const int* sched_progress(const SchedState* st) { return st ? st->d.done_nodes : nullptr; }
void sched_abort(SchedState* st) {
  // from the host, while the kernel runs: a copy on a stream of its own
  if (!st || !st->d_abort) return;
  static const int one = 1;
  cudaStream_t s = nullptr;
  if (cudaStreamCreateWithFlags(&s, cudaStreamNonBlocking)) return;
  cudaMemcpyAsync(st->d_abort, &one, sizeof(int), cudaMemcpyHostToDevice, s);
  cudaStreamSynchronize(s);
  cudaStreamDestroy(s);
}

int sched_job_trace(const SchedState* st, uint64_t* out, int64_t cap, int64_t* njobs) {
  if (njobs) *njobs = st->njobs;
  if (!st->job_trace) return -7;
  if (!out || cap <= 0) return 0;
  std::vector<uint64_t> h((size_t)st->njobs * 4);
  cudaError_t e = cudaMemcpy(h.data(), st->job_trace, h.size() * 8, cudaMemcpyDeviceToHost);
  if (e) return -100 - (int)e;
  for (int64_t j = 0; j < st->njobs && j < cap; ++j) {
    out[5 * j] = h[4 * j];
    out[5 * j + 1] = h[4 * j + 1];
    out[5 * j + 2] = h[4 * j + 2];
    out[5 * j + 3] = ((uint64_t)(uint16_t)st->h_job_type[j] << 32) | (uint32_t)st->h_job_paper[j];
    out[5 * j + 4] = h[4 * j + 3];
  }
  return 0;
}

int sched_job_desc(const SchedState* st, int32_t* out, int64_t cap, int64_t* njobs) {
  if (njobs) *njobs = st->njobs;
  if (!out || cap <= 0) return 0;
  for (int64_t j = 0; j < st->njobs && j < cap; ++j) {
    const Job& jb = st->h_jobs[j];
    int32_t* o = out + 8 * j;
    o[0] = jb.type;
    o[1] = jb.i;
    o[2] = jb.j;
    o[3] = jb.k;
    o[4] = jb.a;
    o[5] = jb.b;
    o[6] = jb.c;
    o[7] = st->h_job_node[j];
  }
  return 0;
}

void sched_destroy(SchedState* st) {
  if (!st) return;
  cudaFree(st->dev_static);
  cudaFree(st->dev_dynamic);
  cudaFree(st->dev_pristine);
  cudaFree(st->job_trace);
  cudaFree(st->d_abort);
  delete st;
}

}  // namespace chol
