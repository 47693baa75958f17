/*
 * chol.h -- C-ABI of the B200-native tiled FP64 Cholesky library (libchol_b200.so).
 *
 * What it computes (Agullo et al., HCW 2015, /root/reference/PAPER.md):
 *   "the Cholesky decomposition of a dense, symmetric, and positive-definite
 *    double-precision matrix A, into the product L L^T, where L is lower
 *    triangular and has positive diagonal elements" (L135-138; A = L L^T,
 *    L166-168), by the tiled right-looking algorithm of Algorithm 1 (L172-181):
 *    the matrix is an N x N grid of nb x nb tiles (L183-186) and four tile
 *    kernels -- POTRF (L196-199), TRSM (L200-202), SYRK (L207-208) and GEMM
 *    (L203-206) -- overwrite A_ij with L_ij in place (L209-211).  Tasks run as
 *    soon as their direct data dependencies (L213-220) are met.
 *
 * Conventions: n = matrix order, nb = tile size,
 * N = n / nb (the paper swaps the letters, reading R1).  All matrices are
 * ROW-MAJOR: element (r, c) of X with leading dimension ld is X[r*ld + c].
 *
 * Status codes: every call returns int; 0 = OK, < 0 = error:
 *   -1  n <= 0
 *   -2  nb <= 0, n % nb != 0, or nb % 32 != 0 (kernel tile granularity)
 *   -3  ngpus < 1, more GPUs than visible devices, or grid_p*grid_q != ngpus
 *   -4  null or misaligned (not 8-byte aligned) pointer, or null plan
 *   -5  lda / ldl < n
 *   -6  bad options (unknown policy / executor / negative values)
 *   -7  chol_trace before any chol_factor*, or tracing disabled
 *   -8  operation not supported for this plan (e.g. chol_solve on a multi-GPU plan)
 *   -9  device out of memory while planning
 *   -10 chol_solve without a successful factorization in the plan
 *   -11 watchdog: the persistent scheduler completed no task node for CHOL_WATCHDOG_S
 *       seconds (env, default 60, 0 = off) -- e.g. a rank of a distributed plan whose
 *       peer never launched; the run is aborted (the kernel exits) and the factor is
 *       incomplete
 *   -100 - e   CUDA runtime error e
 *   (no NCCL codes: the multi-GPU exchange is peer memory, not NCCL)
 * A non-SPD input is NOT an error status: it is reported through *info.
 *
 * Thread safety: a plan may be used by one host thread at a time.
 */
#ifndef CHOL_B200_H
#define CHOL_B200_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct chol_plan_s* chol_plan_t;

/* Scheduling policies of the device-side task scheduler (§V-A,
 * and the static rules of §V-C3). */
enum {
  CHOL_POLICY_CP_PRIORITY = 0, /* (default) ready tasks popped by bottom-level priority (dmdas /
                                  HEFT, L652-660, L299-301) */
  CHOL_POLICY_DYNAMIC = 1,     /* dependency-ready FIFO, any worker (dmda analogue, L645-651) */
  CHOL_POLICY_STATIC = 2       /* CP priority + static placement: POTRF and the TRSMs within
                                  trsm_pin_distance tiles of the diagonal are pinned to the
                                  latency workers; the other TRSMs and all SYRK/GEMM go to the
                                  throughput workers (the paper's TRSM-distance rule,
                                  L1019-1025, transposed to one GPU's two worker classes) */
};

/* Executors. */
enum {
  CHOL_EXEC_SCHEDULER = 0, /* one persistent scheduler kernel per GPU (default) */
  CHOL_EXEC_HOST = 1       /* host-sequenced baseline: per k, POTRF / TRSM batch / update
                              batch launches in Algorithm 1 order (no device scheduler) */
};

/* Options; a zero-initialised struct means "defaults". */
typedef struct {
  int policy;            /* CHOL_POLICY_* (default 0 = CP_PRIORITY, the fastest measured:
                            DYNAMIC is 8% slower at n=28800) */
  int trsm_pin_distance; /* STATIC only: TRSM_i_k with i-k <= d are pinned (0 = default 1:
                            the TRSMs on the POTRF-TRSM-SYRK chain) */
  int latency_workers;   /* STATIC only: CTAs reserved for pinned tasks (0 = default 16) */
  int grid_p, grid_q;    /* 2D block-cyclic process grid (0,0 = the squarest p x q with
                            p <= q for chol_plan; 1 x nranks for chol_plan_dist) */
  int trace;             /* 1 = record per-task t0/t1 (needed by chol_trace);
                            2 = also per-job (CTA sub-task) records (chol_job_trace) */
  int executor;          /* CHOL_EXEC_* */
  int workers;           /* persistent CTAs (0 = one per SM) */
  int cpu_trsm_distance; /* > 0: the host CPU cores are a second resource class -- every
                            TRSM_i_k with i-k >= d runs on them (the paper's static rule,
                            P:L1019-1025, executed in Fig. 11; NEXT-3, DESIGN.md
                            §7f); single-GPU persistent-scheduler plans only (else -6) */
  int cpu_threads;       /* host threads of that class (0 = all host cores) */
} chol_opts_t;

/* One trace record per task (Fig. 12). */
typedef struct {
  uint8_t type;    /* 0 POTRF, 1 TRSM, 2 SYRK, 3 GEMM */
  uint8_t gpu;     /* rank / device that ran it */
  uint16_t worker; /* SM id of the CTA that completed the task's last sub-task */
  int32_t i, j, k; /* Fig. 1 indices: POTRF_k (i=j=k), TRSM_i_k (j=k), SYRK_j_k (i=j), GEMM_i_j_k */
  uint64_t t0_ns;  /* first sub-task start, %globaltimer ns, relative to the factorization start */
  uint64_t t1_ns;  /* last sub-task end */
} chol_task_rec_t;

/* Plan an n x n factorization in nb x nb tiles on ngpus GPUs, the devices
 * 0..ngpus-1 of this process.  ngpus == 1: allocates the tile store (N(N+1)/2 tiles,
 * 8*nb*nb bytes each), the task tables and the scheduler state on the current device.
 * ngpus > 1: one rank of the 2D block-cyclic plan (chol_plan_dist, grid_p x grid_q,
 * default the squarest p <= q) per device, connected in-process through peer memory
 * (NVLink); chol_factor / chol_factor_inplace / chol_generate / chol_scatter /
 * chol_gather / chol_trace fan out to the ranks (A and L: host pointers or device
 * pointers, copied by the owners); chol_solve, chol_run_*, chol_job_trace and the
 * per-rank tile calls return -8.  ngpus > visible devices or grid_p * grid_q != ngpus
 * -> -3.  *out receives the plan; free it with chol_destroy. */
int chol_plan(int64_t n, int64_t nb, int ngpus, chol_plan_t* out);
int chol_plan_ex(int64_t n, int64_t nb, int ngpus, const chol_opts_t* opts, chol_plan_t* out);

/* Factor A = L L^T.  A (lda >= n) and L (ldl >= n) are caller-owned pointers to
 * row-major n x n doubles, either device memory of the plan's GPU or host memory
 * (pinned or pageable; detected with cudaPointerGetAttributes).  Only the lower
 * triangle of A is read.  On return L holds the lower factor with its strictly
 * upper part set to zero.  A == L with lda == ldl (in place) is allowed.
 * Synchronous.  *info (host int) = 0 on success, or j > 0 if the leading minor of
 * order j is not positive definite (1-based global column of the first pivot d
 * with !(d > 0), NaN included); then columns < nb*floor((j-1)/nb) of L are valid
 * and the rest is unspecified. */
int chol_factor(chol_plan_t p, const double* A, int64_t lda, double* L, int64_t ldl, int* info);

/* Per-task trace of the last factorization (requires opts.trace = 1).
 * Copies min(cap, #tasks) records into recs (host memory, may be NULL with
 * cap = 0 to query), sets *nrecs to the number of tasks and *makespan_s to
 * max t1 - min t0 in seconds. */
int chol_trace(chol_plan_t p, chol_task_rec_t* recs, int64_t cap, int64_t* nrecs, double* makespan_s);

/* Per-job (CTA sub-task) trace of the last factorization by the persistent
 * scheduler (requires opts.trace = 2): per job j, out[5j] = t0_ns, out[5j+1] =
 * t1_ns (as chol_trace), out[5j+2] = worker << 32 | SM id, out[5j+4] = time the
 * job was enqueued (its node became ready), out[5j+3] = job type
 * << 32 | dense task id (job types: 0 SYRK/GEMM block, 1 TRSM row slab, 2 POTRF
 * diagonal block, 3 POTRF panel block, 4 POTRF update block, 5 TRSM block solve,
 * 6 TRSM block update, 7 remote-tile receive, 8 diagonal-block inverse (untraced: zero
 * times), 9 no-op).  At most cap jobs; *njobs = number of jobs.  -7 if not available. */
int chol_job_trace(chol_plan_t p, uint64_t* out, int64_t cap, int64_t* njobs);

/* The persistent scheduler's job descriptors, in chol_job_trace's job order (available once
 * the plan exists; tests check the block-level dependencies of the trace with them): per job
 * j, out[8j .. 8j+7] = type (as chol_job_trace), i, j, k (the paper task's tile indices),
 * a, b, c (type-specific: 0 block (bm, bn); 1 row slab; 2 diagonal block b, fused-update
 * flag; 3 inner step b, block row r; 4 inner step b, block (r, q); 5 column block cb, row
 * slab; 6 column block, row slab, target column block; 8 diagonal block b), scheduler node
 * id.  At most cap jobs; *njobs = number of jobs.  -7 without a persistent scheduler, -8 for
 * a multi-GPU plan. */
int chol_job_desc(chol_plan_t p, int32_t* out, int64_t cap, int64_t* njobs);

int chol_destroy(chol_plan_t p);
const char* chol_strerror(int status);

/* ---- helpers for benchmarks / tests (not part of the paper's problem statement) ---- */

/* Fill the plan's tile store in place with a seeded synthetic SPD matrix:
 * family 0 = "uniform" (A_ij = u(i,j) + n [i==j]), family 1 = "integer"
 * (A = L0 L0^T, exact), with the counter-based recipe of DESIGN.md
 * "Input recipe" (same bits as the Python generator spdgen/). */
int chol_generate(chol_plan_t p, uint64_t seed, int family);

/* Copy a row-major matrix (host or device pointer) into / out of the tile store.
 * chol_gather writes L with its strictly upper part zeroed. */
int chol_scatter(chol_plan_t p, const double* A, int64_t lda);
int chol_gather(chol_plan_t p, double* L, int64_t ldl);

/* Host (or device) I/O of the tiles this plan OWNS, packed: `count` nb x nb row-major
 * tiles back to back, in Algorithm 1 tile order (i ascending, then j <= i ascending),
 * restricted to the tiles the rank owns (all N(N+1)/2 tiles on a single-GPU plan;
 * chol_get_dist's nowned on a distributed one) -- the per-rank form of the paper's tile
 * layout, with no n x n host matrix on any rank.  After a
 * factorization the diagonal tiles hold L_kk with zeros above the diagonal.
 * count != the owned-tile count -> -6; null / misaligned pointer -> -4.  Synchronous. */
int chol_scatter_tiles(chol_plan_t p, const double* tiles, int64_t count);
int chol_gather_tiles(chol_plan_t p, double* tiles, int64_t count);

/* Factor the tile store in place (no layout conversion); *info as chol_factor. */
int chol_factor_inplace(chol_plan_t p, int* info);

/* Device time of the last factorization (CUDA events around the launches on the
 * plan's stream) and of the last layout conversion (scatter + gather). */
int chol_last_times(chol_plan_t p, double* factor_s, double* layout_s);

/* The plan's CUDA stream (cudaStream_t) and tile size used by the kernels. */
int chol_get_stream(chol_plan_t p, void** stream);
int chol_get_info(chol_plan_t p, int64_t* n, int64_t* nb, int* block, int* workers, int* policy,
                  int* executor);

/* Run ONE tile task (type 0..3 with Fig. 1 indices i, j, k) on the tile store,
 * alone on the GPU, `reps` times back to back (reps >= 1; for calibration the
 * operands are simply re-used).  Returns the mean device time per run in *ms.
 * Used by the per-kernel parity tests and the calibration of T_t^lat. */
int chol_run_task(chol_plan_t p, int type, int i, int j, int k, int reps, double* ms);

/* Run `count` independent instances of tile task type `type` concurrently
 * (count GEMMs / SYRKs / TRSMs on distinct output tiles of the store, POTRFs on
 * distinct diagonal tiles) and return the device time per instance in *ms
 * (throughput time T_t^thr for a saturating count, latency T_t^lat for count = 1;
 * DESIGN.md reading R9).  Executor CHOL_EXEC_SCHEDULER: the batch runs through the
 * persistent scheduler kernel in the factorization's own job decompositions (count > 1:
 * the bulk forms, row-slab TRSMs; count = 1: the critical-path forms, TRSM column steps
 * and the POTRF block DAG), one untimed warm-up run first; CHOL_EXEC_HOST: one batch
 * launch of the host-executor tile kernels per rep.  Overwrites the store (a factor in
 * it is invalidated).  Errors: -6 bad type, count < 1, reps < 1 or count above the
 * instances available (POTRF N, SYRK N-1, GEMM (N-1)(N-2)/2 at step 0; TRSM N-1 at step 0 on
 * the host executor, N(N-1)/2 panel tiles TRSM_i_k in Algorithm 1 order on the scheduler);
 * -8 on multi-GPU plans. */
int chol_run_batch(chol_plan_t p, int type, int count, int reps, double* ms);

/* ---- multi-GPU: one process (or logical rank) per GPU, 2D block-cyclic owner-computes ----
 * (tile (i,j) lives on rank (i mod p)*q + (j mod q) of the p x q grid,
 * opts->grid_p x opts->grid_q, default 1 x nranks; every task runs on the owner of the tile
 * it overwrites).  A rank stores the tiles it owns plus a cache of the remote panel tiles
 * (L_kk, L_ik) its tasks read; each such tile is pulled once over NVLink by device jobs of
 * the persistent scheduler as soon as its owner publishes it (no host in the loop).
 *
 * chol_plan_dist: plan rank `rank` of `nranks` on the CURRENT device (call cudaSetDevice /
 *   torch.cuda.set_device first).  opts->executor must be CHOL_EXEC_SCHEDULER.
 * chol_dist_export: the rank's connection blob (CUDA IPC handles of its tile store and
 *   publish flags; *len bytes, call with blob = NULL to query the size).
 * chol_dist_connect: blobs = the nranks blobs concatenated in rank order, `stride` bytes
 *   apart (the caller exchanges them, e.g. torch.distributed.all_gather_object).  Blobs
 *   from the same process are used as plain device pointers (logical ranks sharing a
 *   GPU, each with opts->workers CTAs).  Must precede any factorization.
 * chol_generate / chol_scatter / chol_factor* / chol_gather then act on the owned tiles;
 *   *info is this rank's (the global info is the minimum non-zero over ranks).  All
 *   ranks must run the same sequence of factorizations.
 * chol_factor_async / chol_wait: launch / complete a factorization (logical ranks in
 *   one process must all be launched before any wait). */
int chol_plan_dist(int64_t n, int64_t nb, int nranks, int rank, const chol_opts_t* opts, chol_plan_t* out);
int chol_dist_export(chol_plan_t p, void* blob, int64_t cap, int64_t* len);
int chol_dist_connect(chol_plan_t p, const void* blobs, int64_t stride);
int chol_get_dist(chol_plan_t p, int* rank, int* nranks, int* grid_p, int* grid_q, int64_t* nowned, int64_t* nslots);
int chol_factor_async(chol_plan_t p);
int chol_wait(chol_plan_t p, int* info);

/* Solve A X = B with the factor of the plan's last successful chol_factor* (the tiles
 * hold L): L Y = B, then L^T X = Y -- the use of A = L L^T (
 * SURVEY §8f NEXT-2).  B: n x nrhs, ROW-MAJOR with leading dimension ldb >= nrhs, host
 * or device pointer (on the plan's device), caller-owned; overwritten by X.  The call
 * is synchronous.  Method: forward and backward sweeps over bs-row blocks (bs = the
 * plan's block, 96 at nb = 960), each diagonal block applied through its explicit
 * inverse (computed once per factorization, n x bs doubles of plan workspace); the
 * rounding therefore differs from plain substitution.  Single-GPU plans
 * only.  Errors: -4 null / misaligned B or plan, -5 ldb < nrhs, -6 nrhs < 1, -8 a
 * multi-GPU plan, -9 out of memory, -10 no successful factorization (none yet, or the
 * last one reported info > 0), -100 - e CUDA errors. */
int chol_solve(chol_plan_t p, double* B, int64_t ldb, int64_t nrhs);
/* Timing of the last chol_solve: total (copies in/out included) and the two sweeps
 * (plus the diagonal-block inverses when they were recomputed), seconds. */
int chol_last_solve_times(chol_plan_t p, double* total_s, double* sweeps_s);

/* Inject static task priorities into the device scheduler (the paper
 * injects its CP schedules into StarPU): prio[t] for every Algorithm 1 task in
 * chol_task_id order (ntasks = n_tasks(N)), higher runs first -- e.g. minus the start rank of
 * chol_optimal_schedule.  Replaces the bottom-level priority buckets (CHOL_POLICY_CP_PRIORITY /
 * STATIC; pinning kept) for the following factorizations; the factor is unchanged (R15).
 * Errors: -4 null, -6 wrong ntasks, -8 not a persistent-scheduler plan. */
int chol_set_task_priorities(chol_plan_t p, const double* prio, int64_t ntasks);

/* Number of kernel launches the last chol_factor* issued (the persistent scheduler
 * issues 2: queue init + the scheduler kernel). */
int chol_last_launches(chol_plan_t p, int* launches);

/* ---- host-only (no GPU needed) ---- */

/* Task graph of Algorithm 1 for N tiles per side (Fig. 1):
 * *ntasks = N + N(N-1) + N(N-1)(N-2)/6; *nedges = number of direct data
 * dependencies (L213-220); edges[2e], edges[2e+1] = (pred, succ) dense task ids
 * (chol_task_id), at most cap edges written (edges may be NULL). */
int chol_dag(int64_t N, int64_t* ntasks, int64_t* nedges, int64_t* edges, int64_t cap);

/* The host CPU class's TRSM tile kernel (NEXT-3; host only): X (nb x nb, row-major) <- X L^{-T}
 * for the lower triangular L (nb x nb, row-major; only its lower triangle is read), in the
 * inverse form of the device (R19: the inverses of L's bs x bs diagonal blocks by
 * substitution, then two products per column block), AVX-512 when the CPU has it, one thread.
 * Errors: -4 null pointer, -6 nb % bs, nb % 4 or bs % 8 != 0. */
int chol_cpu_trsm(double* X, const double* L, int64_t nb, int bs);

/* Multi-GPU layout of rank `rank` on the p x q grid (host only): *nowned tiles owned,
 * *ncached remote panel tiles received; slot_map[t] (t = i(i+1)/2 + j, at most cap
 * entries, may be NULL) = local slot of tile t (owned: [0, nowned) in tile order; cached:
 * [nowned, nowned + ncached) in order of first use), -1 if absent. */
int chol_dist_layout(int64_t n, int64_t nb, int p, int q, int rank, int* nowned, int* ncached, int32_t* slot_map,
                     int64_t cap);

/* Dense id of task (type, i, j, k) in chol_dag / chol_trace numbering. */
int chol_task_id(int64_t N, int type, int i, int j, int k, int64_t* id);

/* Makespan lower bounds of PAPER.md §III (L334-408, L495-502) for one resource type
 * (ngpus GPUs), from per-type latency times T_lat[4] (a task alone on an idle GPU)
 * and throughput times T_thr[4] (per task in a saturating batch), indexed
 * POTRF, TRSM, SYRK, GEMM, in seconds.  out[0] area = sum_t N_t T_thr_t / M,
 * out[1] chain = N T_lat_P + (N-1)(T_lat_T + T_lat_S), out[2] mixed = max(area,
 * chain), out[3] critical path (longest DAG path, T_lat weights; -1 if N > 256),
 * out[4] GEMM-peak bound (n^3/3) / (M 2 nb^3 / T_thr_G), out[5] max(area, cp). */
int chol_bounds(int64_t n, int64_t nb, int ngpus, const double* T_lat, const double* T_thr, double* out);

/* Owner-area bound (ext; host only): on a p x q 2D block-cyclic grid with
 * owner-computes every task runs on the owner of the tile it overwrites, so
 * no schedule beats the busiest rank: *out = max_g sum_{tasks of g} T_thr[type] (seconds,
 * T_thr as in chol_bounds).  per_rank (may be NULL) receives the p*q sums.  Errors: -1
 * N <= 0, -3 p or q < 1, -4 null pointer. */
int chol_owner_area(int64_t N, int p, int q, const double* T_thr, double* out, double* per_rank);

/* ---- platform model (host only): the paper's LP bounds over several resource types and
 * its scheduler simulation (§III-A, §IV-C, §V;
 * SURVEY §8f NEXT-1).  Times are per task of each type on one processing element of a
 * class, in seconds; a negative or infinite time means the class cannot run that type. */
#define CHOL_SIM_MAX_CLASSES 4

/* LP of L349-359 (area bound; mixed != 0 adds the chain constraint of L390-396:
 *   sum_r n_rP T_rP + (N-1) T*_T + (N-1) T*_S <= l, T* = fastest time over the classes)
 * over nclasses resource types with workers[r] processing elements and times
 * time[r*4 + t] (t = POTRF, TRSM, SYRK, GEMM).  The n_rt are relaxed to reals (reading
 * R10).  *l = optimal makespan bound; n_rt (may be NULL) = optimal task counts per class
 * and type (row-major nclasses x 4).  Errors: -1 N <= 0; -6 bad arguments or a task type
 * no class can run. */
int chol_lp_bound(int64_t N, int nclasses, const int* workers, const double* time, int mixed, double* l,
                  double* n_rt);

/* Scheduler policies of the simulation (StarPU's, L645-660). */
enum {
  CHOL_SIM_DMDA = 0,  /* ready tasks (release order) go to the worker with the minimum estimated
                         completion time; each worker runs its queue in FIFO order */
  CHOL_SIM_DMDAS = 1, /* the same, ready tasks and worker queues in bottom-level priority order
                         (longest path to an exit task with each type's fastest time, L655-660) */
  CHOL_SIM_FIXED = 2  /* an injected static schedule (the paper's CP schedule replayed in
                         simulation, L1056-1072): task t runs on worker fixed_worker[t], each worker
                         runs its tasks in increasing fixed_rank[t] order, each as soon as its
                         predecessors have finished and the worker is free */
};
typedef struct {
  int nclasses;                            /* 1 .. CHOL_SIM_MAX_CLASSES */
  int workers[CHOL_SIM_MAX_CLASSES];       /* processing elements per class */
  double time[CHOL_SIM_MAX_CLASSES][4];    /* seconds per task, [class][POTRF, TRSM, SYRK, GEMM] */
  int policy;                              /* CHOL_SIM_DMDA / CHOL_SIM_DMDAS */
  int gemm_syrk_class;                     /* static rule (L1000-1007): SYRK/GEMM only on this class; -1 off */
  int trsm_far_class;                      /* static rule (L1019-1025): TRSM_i_k with i-k >= */
  int trsm_far_distance;                   /*   trsm_far_distance only on trsm_far_class; -1 off */
  const int32_t* fixed_worker;             /* CHOL_SIM_FIXED: worker per task (chol_task_id order) */
  const int32_t* fixed_rank;               /* CHOL_SIM_FIXED: order of the task on its worker */
} chol_sim_opts_t;

/* Discrete-event replay of the Algorithm 1 task DAG for N tiles per side on the
 * platform described by *opts (no data transfers modelled, reading R18).  Ties: events
 * at equal times are processed together; a task goes to the lowest-numbered worker among
 * equal completion times; workers are numbered class by class.  *makespan in seconds;
 * recs (may be NULL; at most cap written, indexed by chol_task_id) receive each task's
 * class (field gpu), worker, and t0/t1 in ns.  Errors: -1 N <= 0, -4 null pointer,
 * -6 bad options or a task no class may run. */
int chol_simulate(int64_t N, const chol_sim_opts_t* opts, double* makespan, chol_task_rec_t* recs, int64_t cap);

/* Exact minimum-makespan schedule of the Algorithm 1 DAG for small N (the
 * paper's constraint-programming formulation, P:L409-464 -- one resource class per task,
 * start times, cumulative resource limits, dependencies, no transfers -- solved to proven
 * optimality where the paper's CP Optimizer ran 23 hours without a proof).
 * Method: depth-first branch and bound over semi-active schedules generated in order of start
 * time (every schedule can be left-shifted to a semi-active one, so one of them is optimal);
 * identical workers of a class are interchangeable (a task goes to a worker of its class free
 * earliest); bounds: the longest remaining path with each type's fastest time, the remaining
 * work over all workers; initial incumbent: the dmdas replay.  The platform, the static rules
 * and the times are those of *opts (policy and fixed_* ignored).  Outputs: *makespan;
 * *optimal = 1 if the search completed, 0 if node_limit (0 = 2e8) stopped it first (the best
 * schedule found is returned); worker / rank (may be NULL; n_tasks entries, chol_task_id
 * order) -- a schedule CHOL_SIM_FIXED replays; *nodes = search nodes.  Errors: -1 N <= 0,
 * -4 null pointer, -6 bad options, a task no class may run, or N > 8. */
int chol_optimal_schedule(int64_t N, const chol_sim_opts_t* opts, int64_t node_limit, double* makespan,
                          int* optimal, int32_t* worker, int32_t* rank, int64_t* nodes);

#ifdef __cplusplus
}
#endif
#endif /* CHOL_B200_H */
