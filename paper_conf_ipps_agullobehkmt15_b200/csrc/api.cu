// C-ABI of libchol_b200.so (include/chol.h): planner, layout conversion, executors.
#include <cuda.h>
#include <cuda_runtime.h>

#include <algorithm>
#include <climits>
#include <cstdio>
#include <cstring>
#include <new>
#include <thread>
#include <vector>

#include "../../include/chol.h"
#include "kernels.h"
#include "sched.h"
#include "taskid.h"

using namespace chol;

struct chol_plan_s {
  int64_t n = 0, nb = 0, N = 0, ntiles = 0, ntasks = 0;
  int bs = 0, device = 0, ngpus = 1, sms = 0;
  chol_opts_t opts{};
  cudaStream_t stream = nullptr;
  double* tiles = nullptr;
  CUtensorMap map{};
  int* d_info = nullptr;
  uint64_t* d_base = nullptr;
  uint64_t* d_t0 = nullptr;
  uint64_t* d_t1 = nullptr;
  cudaEvent_t ev0 = nullptr, ev1 = nullptr, ev2 = nullptr, ev3 = nullptr;
  double last_factor_s = 0.0, last_layout_s = 0.0;
  bool factored = false;
  int last_launches = 0;
  SchedState* sched = nullptr;  // persistent-scheduler state (sched.cu)
};

#define CUDA_TRY(x)                                   \
  do {                                                \
    cudaError_t e_ = (x);                             \
    if (e_ != cudaSuccess) return -100 - (int)e_;     \
  } while (0)

// ------------------------------------------------------------------ TMA map
typedef CUresult (*PFN_encodeTiled_t)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*,
                                      const cuuint64_t*, const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave,
                                      CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

static int encode_tile_map(chol_plan_s* p) {
  void* fn = nullptr;
  cudaDriverEntryPointQueryResult q;
  CUDA_TRY(cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fn, cudaEnableDefault, &q));
  if (!fn || q != cudaDriverEntryPointSuccess) return -100 - (int)cudaErrorNotSupported;
  auto encode = reinterpret_cast<PFN_encodeTiled_t>(fn);
  const cuuint64_t dims[3] = {(cuuint64_t)p->nb, (cuuint64_t)p->nb, (cuuint64_t)p->ntiles};
  const cuuint64_t strides[2] = {(cuuint64_t)p->nb * 8, (cuuint64_t)p->nb * p->nb * 8};
  const cuuint32_t box[3] = {16, (cuuint32_t)p->bs, 1};
  const cuuint32_t estr[3] = {1, 1, 1};
  CUresult r = encode(&p->map, CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 3, p->tiles, dims, strides, box, estr,
                      CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_128B, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                      CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  if (r != CUDA_SUCCESS) return -100 - (int)cudaErrorInvalidValue;
  return 0;
}

// ------------------------------------------------------------------ errors
extern "C" const char* chol_strerror(int s) {
  switch (s) {
    case 0: return "success";
    case -1: return "n <= 0";
    case -2: return "nb <= 0, n % nb != 0, or nb % 32 != 0";
    case -3: return "bad ngpus or process grid";
    case -4: return "null or misaligned pointer / plan";
    case -5: return "leading dimension < n";
    case -6: return "bad options";
    case -7: return "no trace available (factor first with opts.trace = 1)";
    case -8: return "not supported by this build";
    case -9: return "device out of memory";
  }
  if (s <= -200) return "NCCL error";
  if (s <= -100) return cudaGetErrorString((cudaError_t)(-100 - s));
  return "unknown status";
}

static int pick_block(int64_t nb) {
  if (nb % 96 == 0) return 96;
  if (nb % 64 == 0) return 64;
  if (nb % 32 == 0) return 32;
  return 0;
}

// ------------------------------------------------------------------ plan
extern "C" int chol_destroy(chol_plan_t p) {
  if (!p) return -4;
  if (p->sched) sched_destroy(p->sched);
  cudaSetDevice(p->device);
  if (p->stream) cudaStreamSynchronize(p->stream);
  cudaFree(p->tiles);
  cudaFree(p->d_info);
  cudaFree(p->d_base);
  cudaFree(p->d_t0);
  cudaFree(p->d_t1);
  if (p->ev0) cudaEventDestroy(p->ev0);
  if (p->ev1) cudaEventDestroy(p->ev1);
  if (p->ev2) cudaEventDestroy(p->ev2);
  if (p->ev3) cudaEventDestroy(p->ev3);
  if (p->stream) cudaStreamDestroy(p->stream);
  delete p;
  return 0;
}

extern "C" int chol_plan_ex(int64_t n, int64_t nb, int ngpus, const chol_opts_t* o, chol_plan_t* out) {
  if (!out) return -4;
  *out = nullptr;
  if (n <= 0) return -1;
  if (nb <= 0 || n % nb != 0 || nb % 32 != 0) return -2;
  chol_opts_t opts{};
  if (o) opts = *o;
  if (opts.policy < 0 || opts.policy > 2 || opts.executor < 0 || opts.executor > 1 || opts.trsm_pin_distance < 0 ||
      opts.latency_workers < 0 || opts.workers < 0 || opts.grid_p < 0 || opts.grid_q < 0 || opts.trace < 0 ||
      opts.trace > 2)
    return -6;
  int ndev = 0;
  if (cudaGetDeviceCount(&ndev) != cudaSuccess) ndev = 0;
  if (ngpus < 1 || ngpus > ndev) return -3;
  if (opts.grid_p == 0 && opts.grid_q == 0) {
    opts.grid_p = 1;
    opts.grid_q = ngpus;
  }
  if (opts.grid_p * opts.grid_q != ngpus) return -3;
  if (ngpus > 1) return -8;  // multi-GPU runs one process per GPU (chol_plan_dist)

  auto* p = new (std::nothrow) chol_plan_s();
  if (!p) return -9;
  p->n = n;
  p->nb = nb;
  p->N = n / nb;
  p->ntiles = p->N * (p->N + 1) / 2;
  p->ntasks = n_tasks(p->N);
  p->bs = pick_block(nb);
  p->opts = opts;
  p->ngpus = ngpus;
  int st = 0;
  auto fail = [&](int s) {
    chol_destroy(p);
    return s;
  };
  if ((st = -100 - (int)cudaGetDevice(&p->device)) != -100) return fail(st);
  cudaSetDevice(p->device);
  cudaDeviceGetAttribute(&p->sms, cudaDevAttrMultiProcessorCount, p->device);
  if (p->ntiles > INT_MAX) return fail(-2);
  const size_t bytes = (size_t)p->ntiles * nb * nb * sizeof(double);
  cudaError_t e = cudaMalloc(&p->tiles, bytes);
  if (e == cudaErrorMemoryAllocation) {
    cudaGetLastError();
    return fail(-9);
  }
  if (e) return fail(-100 - (int)e);
  if ((e = cudaStreamCreateWithFlags(&p->stream, cudaStreamNonBlocking))) return fail(-100 - (int)e);
  if ((e = cudaMalloc(&p->d_info, sizeof(int)))) return fail(-100 - (int)e);
  if ((e = cudaMalloc(&p->d_base, sizeof(uint64_t)))) return fail(-100 - (int)e);
  if (opts.trace) {
    if ((e = cudaMalloc(&p->d_t0, p->ntasks * sizeof(uint64_t)))) return fail(-100 - (int)e);
    if ((e = cudaMalloc(&p->d_t1, p->ntasks * sizeof(uint64_t)))) return fail(-100 - (int)e);
  }
  for (cudaEvent_t* ev : {&p->ev0, &p->ev1, &p->ev2, &p->ev3})
    if ((e = cudaEventCreate(ev))) return fail(-100 - (int)e);
  if ((st = encode_tile_map(p))) return fail(st);
  if ((e = prepare_kernels(p->bs))) return fail(-100 - (int)e);
  if (opts.executor == CHOL_EXEC_SCHEDULER) {
    if ((st = sched_create(&p->sched, p->N, p->nb, p->bs, p->sms, &p->opts, p->stream))) return fail(st);
  }
  *out = p;
  return 0;
}

extern "C" int chol_plan(int64_t n, int64_t nb, int ngpus, chol_plan_t* out) {
  return chol_plan_ex(n, nb, ngpus, nullptr, out);
}

extern "C" int chol_get_stream(chol_plan_t p, void** stream) {
  if (!p || !stream) return -4;
  *stream = (void*)p->stream;
  return 0;
}

extern "C" int chol_get_info(chol_plan_t p, int64_t* n, int64_t* nb, int* block, int* workers, int* policy,
                             int* executor) {
  if (!p) return -4;
  if (n) *n = p->n;
  if (nb) *nb = p->nb;
  if (block) *block = p->bs;
  if (workers) *workers = p->sched ? sched_workers(p->sched) : 0;
  if (policy) *policy = p->opts.policy;
  if (executor) *executor = p->opts.executor;
  return 0;
}

// ------------------------------------------------------------------ layout
static bool is_device_ptr(const void* ptr) {
  cudaPointerAttributes a{};
  if (cudaPointerGetAttributes(&a, ptr) != cudaSuccess) {
    cudaGetLastError();
    return false;
  }
  return a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged;
}

static int scatter_impl(chol_plan_s* p, const double* A, int64_t lda) {
  const int64_t nb = p->nb;
  for (int64_t i = 0; i < p->N; ++i)
    for (int64_t j = 0; j <= i; ++j) {
      double* dst = p->tiles + tile_index((int)i, (int)j) * nb * nb;
      const double* src = A + i * nb * lda + j * nb;
      CUDA_TRY(cudaMemcpy2DAsync(dst, nb * 8, src, lda * 8, nb * 8, nb, cudaMemcpyDefault, p->stream));
    }
  return 0;
}

static void host_zero_upper_tiles(double* L, int64_t ldl, int64_t n, int64_t nb) {
  // strictly-upper tiles (column tiles right of the diagonal tile), multithreaded
  const int64_t N = n / nb;
  unsigned nt = std::max(1u, std::min(16u, std::thread::hardware_concurrency()));
  std::vector<std::thread> th;
  for (unsigned w = 0; w < nt; ++w)
    th.emplace_back([=] {
      for (int64_t r = w; r < n; r += nt) {
        const int64_t c0 = (r / nb + 1) * nb;
        if (c0 < n) memset(L + r * ldl + c0, 0, (size_t)(n - c0) * sizeof(double));
      }
    });
  for (auto& t : th) t.join();
  (void)N;
}

static int gather_impl(chol_plan_s* p, double* L, int64_t ldl) {
  const int64_t nb = p->nb, n = p->n;
  CUDA_TRY(launch_zero_upper_diag(p->tiles, (int)nb, (int)p->N, p->stream));
  const bool dev = is_device_ptr(L);
  for (int64_t i = 0; i < p->N; ++i) {
    for (int64_t j = 0; j <= i; ++j) {
      const double* src = p->tiles + tile_index((int)i, (int)j) * nb * nb;
      double* dst = L + i * nb * ldl + j * nb;
      CUDA_TRY(cudaMemcpy2DAsync(dst, ldl * 8, src, nb * 8, nb * 8, nb, cudaMemcpyDefault, p->stream));
    }
    if (dev && (i + 1) * nb < n)
      CUDA_TRY(cudaMemset2DAsync(L + i * nb * ldl + (i + 1) * nb, ldl * 8, 0, (n - (i + 1) * nb) * 8, nb, p->stream));
  }
  if (!dev) host_zero_upper_tiles(L, ldl, n, nb);
  return 0;
}

extern "C" int chol_scatter(chol_plan_t p, const double* A, int64_t lda) {
  if (!p || !A || (reinterpret_cast<uintptr_t>(A) & 7)) return -4;
  if (lda < p->n) return -5;
  cudaSetDevice(p->device);
  int st = scatter_impl(p, A, lda);
  if (st) return st;
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  return 0;
}

extern "C" int chol_gather(chol_plan_t p, double* L, int64_t ldl) {
  if (!p || !L || (reinterpret_cast<uintptr_t>(L) & 7)) return -4;
  if (ldl < p->n) return -5;
  cudaSetDevice(p->device);
  int st = gather_impl(p, L, ldl);
  if (st) return st;
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  return 0;
}

extern "C" int chol_generate(chol_plan_t p, uint64_t seed, int family) {
  if (!p) return -4;
  if (family < 0 || family > 1) return -6;
  cudaSetDevice(p->device);
  CUDA_TRY(launch_generate(p->tiles, p->n, (int)p->nb, (int)p->N, seed, family, p->stream));
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  return 0;
}

// ------------------------------------------------------------------ executors
static StepParams base_params(chol_plan_s* p) {
  StepParams sp{};
  sp.tiles = p->tiles;
  sp.nb = (int)p->nb;
  sp.N = (int)p->N;
  sp.info = p->d_info;
  if (p->opts.trace) {
    sp.tr_t0 = p->d_t0;
    sp.tr_t1 = p->d_t1;
    sp.tr_base = p->d_base;
  }
  return sp;
}

// Algorithm 1 in program order, one batch launch per (k, kernel type).
static int run_host_sequenced(chol_plan_s* p, int* nlaunch) {
  StepParams sp = base_params(p);
  const int N = (int)p->N;
  for (int k = 0; k < N; ++k) {
    sp.k = k;
    CUDA_TRY(launch_potrf(p->bs, p->map, sp, 1, p->stream, nlaunch));
    if (k == N - 1) break;
    sp.i0 = k + 1;
    CUDA_TRY(launch_trsm(p->bs, p->map, sp, N - 1 - k, p->stream, nlaunch));
    const int m = N - 1 - k;
    sp.mode = 0;
    CUDA_TRY(launch_update(p->bs, p->map, sp, m * (m + 1) / 2, p->stream, nlaunch));
  }
  return 0;
}

static int factor_launch(chol_plan_s* p) {
  CUDA_TRY(launch_init_info(p->d_info, p->stream));
  if (p->opts.trace) {
    CUDA_TRY(cudaMemsetAsync(p->d_t0, 0xff, p->ntasks * sizeof(uint64_t), p->stream));
    CUDA_TRY(cudaMemsetAsync(p->d_t1, 0, p->ntasks * sizeof(uint64_t), p->stream));
  }
  CUDA_TRY(launch_stamp(p->d_base, p->stream));
  int nl = 0;
  CUDA_TRY(cudaEventRecord(p->ev0, p->stream));
  int st = 0;
  if (p->opts.executor == CHOL_EXEC_HOST)
    st = run_host_sequenced(p, &nl);
  else
    st = sched_run(p->sched, p->map, base_params(p), p->stream, &nl);
  if (st) return st;
  CUDA_TRY(cudaEventRecord(p->ev1, p->stream));
  p->last_launches = nl;
  return 0;
}

static int finish_info(chol_plan_s* p, int* info) {
  int h = 0;
  CUDA_TRY(cudaMemcpyAsync(&h, p->d_info, sizeof(int), cudaMemcpyDeviceToHost, p->stream));
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  float ms = 0.f;
  CUDA_TRY(cudaEventElapsedTime(&ms, p->ev0, p->ev1));
  p->last_factor_s = ms * 1e-3;
  p->factored = true;
  if (info) *info = (h == INT_MAX) ? 0 : h;
  return 0;
}

extern "C" int chol_factor_inplace(chol_plan_t p, int* info) {
  if (!p) return -4;
  cudaSetDevice(p->device);
  int st = factor_launch(p);
  if (st) return st;
  return finish_info(p, info);
}

extern "C" int chol_factor(chol_plan_t p, const double* A, int64_t lda, double* L, int64_t ldl, int* info) {
  if (!p || !A || !L || (reinterpret_cast<uintptr_t>(A) & 7) || (reinterpret_cast<uintptr_t>(L) & 7)) return -4;
  if (lda < p->n || ldl < p->n) return -5;
  cudaSetDevice(p->device);
  CUDA_TRY(cudaEventRecord(p->ev2, p->stream));
  int st = scatter_impl(p, A, lda);
  if (st) return st;
  if ((st = factor_launch(p))) return st;
  if ((st = gather_impl(p, L, ldl))) return st;
  CUDA_TRY(cudaEventRecord(p->ev3, p->stream));
  if ((st = finish_info(p, info))) return st;
  float tot = 0.f;
  CUDA_TRY(cudaEventElapsedTime(&tot, p->ev2, p->ev3));
  p->last_layout_s = tot * 1e-3 - p->last_factor_s;
  return 0;
}

extern "C" int chol_last_launches(chol_plan_t p, int* launches) {
  if (!p || !launches) return -4;
  *launches = p->last_launches;
  return 0;
}

extern "C" int chol_last_times(chol_plan_t p, double* factor_s, double* layout_s) {
  if (!p) return -4;
  if (factor_s) *factor_s = p->last_factor_s;
  if (layout_s) *layout_s = p->last_layout_s;
  return 0;
}

// ------------------------------------------------------------------ trace
extern "C" int chol_trace(chol_plan_t p, chol_task_rec_t* recs, int64_t cap, int64_t* nrecs, double* makespan_s) {
  if (!p) return -4;
  if (!p->opts.trace || !p->factored) return -7;
  cudaSetDevice(p->device);
  std::vector<uint64_t> t0(p->ntasks), t1(p->ntasks);
  CUDA_TRY(cudaMemcpy(t0.data(), p->d_t0, p->ntasks * 8, cudaMemcpyDeviceToHost));
  CUDA_TRY(cudaMemcpy(t1.data(), p->d_t1, p->ntasks * 8, cudaMemcpyDeviceToHost));
  const int64_t N = p->N;
  uint64_t lo = UINT64_MAX, hi = 0;
  int64_t w = 0;
  auto emit = [&](int type, int i, int j, int k, int64_t id) {
    const uint64_t a = t0[id], b = t1[id] >> 16;
    if (t0[id] != UINT64_MAX) {
      lo = std::min(lo, a);
      hi = std::max(hi, b);
    }
    if (recs && w < cap) {
      chol_task_rec_t& r = recs[w];
      r.type = (uint8_t)type;
      r.gpu = 0;
      r.worker = (uint16_t)(t1[id] & 0xffff);
      r.i = i;
      r.j = j;
      r.k = k;
      r.t0_ns = a;
      r.t1_ns = b;
    }
    ++w;
  };
  // records in Algorithm 1 order
  for (int k = 0; k < N; ++k) {
    emit(T_POTRF, k, k, k, id_potrf(N, k));
    for (int i = k + 1; i < N; ++i) emit(T_TRSM, i, k, k, id_trsm(N, i, k));
    for (int j = k + 1; j < N; ++j) {
      emit(T_SYRK, j, j, k, id_syrk(N, j, k));
      for (int i = j + 1; i < N; ++i) emit(T_GEMM, i, j, k, id_gemm(N, i, j, k));
    }
  }
  if (nrecs) *nrecs = w;
  if (makespan_s) *makespan_s = (hi > lo) ? (hi - lo) * 1e-9 : 0.0;
  return 0;
}

extern "C" int chol_job_trace(chol_plan_t p, uint64_t* out, int64_t cap, int64_t* njobs) {
  if (!p) return -4;
  if (!p->sched || p->opts.trace != 2 || !p->factored) return -7;
  cudaSetDevice(p->device);
  return sched_job_trace(p->sched, out, cap, njobs);  // 5 u64 per job
}

// ------------------------------------------------------------------ calibration / single tasks
extern "C" int chol_run_task(chol_plan_t p, int type, int i, int j, int k, int reps, double* ms) {
  if (!p) return -4;
  const int N = (int)p->N;
  if (type < 0 || type > 3 || reps < 1 || k < 0 || k >= N) return -6;
  if (type == T_TRSM && !(i > k && i < N)) return -6;
  if (type == T_SYRK && !(j > k && j < N)) return -6;
  if (type == T_GEMM && !(i > j && j > k && i < N)) return -6;
  cudaSetDevice(p->device);
  StepParams sp = base_params(p);
  sp.tr_t0 = sp.tr_t1 = nullptr;
  sp.tr_base = nullptr;
  sp.k = k;
  CUDA_TRY(launch_init_info(p->d_info, p->stream));
  CUDA_TRY(cudaEventRecord(p->ev0, p->stream));
  int nl = 0;
  for (int r = 0; r < reps; ++r) {
    if (type == T_POTRF) {
      CUDA_TRY(launch_potrf(p->bs, p->map, sp, 1, p->stream, &nl));
    } else if (type == T_TRSM) {
      sp.i0 = i;
      CUDA_TRY(launch_trsm(p->bs, p->map, sp, 1, p->stream, &nl));
    } else {
      sp.mode = 1;
      sp.i0 = (type == T_SYRK) ? j : i;
      sp.j0 = j;
      CUDA_TRY(launch_update(p->bs, p->map, sp, 1, p->stream, &nl));
    }
  }
  CUDA_TRY(cudaEventRecord(p->ev1, p->stream));
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  float t = 0.f;
  CUDA_TRY(cudaEventElapsedTime(&t, p->ev0, p->ev1));
  if (ms) *ms = t / reps;
  return 0;
}

extern "C" int chol_run_batch(chol_plan_t p, int type, int count, int reps, double* ms) {
  if (!p) return -4;
  const int N = (int)p->N;
  if (type < 0 || type > 3 || reps < 1 || count < 1) return -6;
  // instances at step k = 0: POTRF on diagonal tiles 0..count-1, TRSM (i, 0),
  // SYRK (j, 0), GEMM (i, j, 0) -- all with distinct output tiles.
  const int maxc = type == T_POTRF ? N : type == T_GEMM ? (N - 1) * (N - 2) / 2 : N - 1;
  if (count > maxc) return -6;
  cudaSetDevice(p->device);
  StepParams sp = base_params(p);
  sp.tr_t0 = sp.tr_t1 = nullptr;
  sp.tr_base = nullptr;
  sp.k = 0;
  CUDA_TRY(launch_init_info(p->d_info, p->stream));
  CUDA_TRY(cudaEventRecord(p->ev0, p->stream));
  int nl = 0;
  for (int r = 0; r < reps; ++r) {
    if (type == T_POTRF) {
      CUDA_TRY(launch_potrf(p->bs, p->map, sp, count, p->stream, &nl));
    } else if (type == T_TRSM) {
      sp.i0 = 1;
      CUDA_TRY(launch_trsm(p->bs, p->map, sp, count, p->stream, &nl));
    } else {
      sp.mode = type == T_GEMM ? 2 : 3;
      CUDA_TRY(launch_update(p->bs, p->map, sp, count, p->stream, &nl));
    }
  }
  CUDA_TRY(cudaEventRecord(p->ev1, p->stream));
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  float t = 0.f;
  CUDA_TRY(cudaEventElapsedTime(&t, p->ev0, p->ev1));
  if (ms) *ms = t / reps / count;
  return 0;
}
