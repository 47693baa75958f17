// Device-side dependency-counting task scheduler (CHOL_EXEC_SCHEDULER).
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>

#include <utility>
#include <vector>

#include "../../include/chol.h"
#include "kernels.h"

namespace chol {
struct SchedState;

// Multi-GPU (2D block-cyclic owner-computes): what this rank owns.
struct DistInfo {
  int p, q, rank, nranks;
  const int* h_slot_map;  // host, N(N+1)/2 entries: local slot of tile t (owned or cached), -1 = absent
};
__host__ __device__ inline int tile_owner(int i, int j, int p, int q) { return (i % p) * q + (j % q); }

int sched_create(SchedState** out, int64_t N, int64_t nb, int bs, int sms, const chol_opts_t* opts, cudaStream_t s,
                 const DistInfo* dist = nullptr);
// calibration batch: `count` independent tasks of one type (T_POTRF..T_GEMM) at step 0 on
// distinct output tiles, run by the persistent kernel (chol_run_batch); -6 bad type / count
int sched_create_batch(SchedState** out, int64_t N, int64_t nb, int bs, int sms, const chol_opts_t* opts, int type,
                       int count);
// Dinv workspace of the inverse-form TRSM slabs: [N][nb/bs] bs x bs blocks (plan-owned) and
// its TMA map (dims {bs, bs, N nb/bs}, box {16, bs, 1}, 128B swizzle)
int sched_set_dinv(SchedState* st, double* dinv, const CUtensorMap& dmap);
// the TRSM_i_k (i, k) this plan runs on the host CPU class (opts->cpu_trsm_distance)
const std::vector<std::pair<int, int>>& sched_host_tasks(const SchedState* st);
// injected static priorities per Algorithm 1 task (higher first; NEXT-4)
int sched_set_priorities(SchedState* st, const double* prio, int64_t ntasks);
// device pointers of the distributed plan, known after the IPC handle exchange
int sched_set_dist(SchedState* st, const int* d_slot_map, const int* d_owner_slot, double* const* d_peer_slots,
                   int* const* d_peer_flags, int* d_my_flags);
int sched_run(SchedState* st, const CUtensorMap& map, const StepParams& base, cudaStream_t s, int* nlaunch,
              unsigned epoch = 1);
int sched_workers(const SchedState* st);
// device counter of completed nodes (host watchdog, api.cu)
const int* sched_progress(const SchedState* st);
// stop a stalled run: the scheduler warps hand out no further jobs and the kernel exits
void sched_abort(SchedState* st);
// Streamed input (chol_factor from host memory): the order in which the tiles are copied
// in, which the scheduler's watch list follows (fixed when the plan is built).
void sched_arrival_order(const SchedState* st, std::vector<std::pair<int, int>>& tiles);
int sched_job_trace(const SchedState* st, uint64_t* out, int64_t cap, int64_t* njobs);
int sched_job_desc(const SchedState* st, int32_t* out, int64_t cap, int64_t* njobs);
void sched_destroy(SchedState* st);
// development: print the CHOL_PHASES job-phase counters (no-op in normal builds)
void sched_phase_dump();
}  // namespace chol
