// C-ABI of libchol_b200.so (include/chol.h): planner, layout conversion, executors.
#include <cuda.h>
#include <cuda_runtime.h>

#include <algorithm>
#include <climits>
#include <cstdio>
#include <cstring>
#include <new>
#include <thread>
#include <chrono>
#include <vector>

#include <unistd.h>

#include "../../include/chol.h"
#include "dag.h"
#include "hetero.h"
#include "kernels.h"
#include "sched.h"
#include "solve.h"
#include "taskid.h"

using namespace chol;

struct chol_plan_s {
  int64_t n = 0, nb = 0, N = 0, ntiles = 0, ntasks = 0;
  int bs = 0, device = 0, ngpus = 1, sms = 0;
  chol_opts_t opts{};
  cudaStream_t stream = nullptr;
  double* tiles = nullptr;
  CUtensorMap map{};
  double* d_dinv = nullptr;  // inverse-form TRSM: inverses of the diagonal blocks of every L_kk
  CUtensorMap dmap{};
  int* d_info = nullptr;
  uint64_t* d_base = nullptr;
  uint64_t* d_t0 = nullptr;
  uint64_t* d_t1 = nullptr;
  cudaEvent_t ev0 = nullptr, ev1 = nullptr, ev2 = nullptr, ev3 = nullptr;
  double last_factor_s = 0.0, last_layout_s = 0.0;
  bool factored = false;
  int last_launches = 0;
  SchedState* sched = nullptr;  // persistent-scheduler state (sched.cu)
  // ---- multi-GPU (chol_plan_dist): this rank's share of the 2D block-cyclic layout
  bool dist = false, connected = false;
  int rank = 0, nranks = 1, p = 1, q = 1;
  int64_t nslots = 0, nowned = 0;
  std::vector<int> h_slot_map, h_owned_tile;  // tile -> local slot; owned slot -> tile
  int* d_slot_map = nullptr;
  int* d_owner_slot = nullptr;
  int* d_owned_tile = nullptr;
  int* d_diag_slots = nullptr;  // owned diagonal tiles' slots
  int ndiag = 0;
  int* d_flags = nullptr;       // per tile: epoch in which this rank published it
  double** d_peer_slots = nullptr;
  int** d_peer_flags = nullptr;
  std::vector<void*> ipc_opened;
  unsigned epoch = 0;
  // ---- single GPU, persistent scheduler: streamed host input / output (chol_factor)
  int* d_in_flags = nullptr;   // per tile: epoch in which its input copy landed (device)
  int* h_out_flags = nullptr;  // per tile: epoch in which it became final (host-mapped); second half:
                               // epoch in which a host-class TRSM's inputs became final
  int* d_host_flags = nullptr; // per tile: epoch in which the host class wrote L_ik back (device)
  HostTrsm* host = nullptr;    // host CPU class (opts.cpu_trsm_distance > 0)
  int* d_out_flags = nullptr;  // device alias of h_out_flags
  int* h_epoch = nullptr;      // pinned source of the 4-byte arrival-flag copies
  cudaStream_t s_in = nullptr, s_out = nullptr;
  bool streamed_run = false;
  // ---- triangular solves with the factor (chol_solve, solve.cu)
  int last_info = -1;           // info of the last completed factorization (-1: none)
  double* d_inv = nullptr;      // diagonal-block inverses + chain matrices (3 n x bs doubles)
  bool inv_valid = false;
  double* d_rhs = nullptr;      // padded right-hand sides, n x ldw
  size_t rhs_cap = 0;           // doubles
  int* d_solve_ctl = nullptr;   // counters + flags
  size_t ctl_cap = 0;           // ints
  double last_solve_s = 0.0, last_sweeps_s = 0.0;
  cudaEvent_t ev4 = nullptr, ev5 = nullptr;
  // ---- one process driving ngpus devices (chol_plan with ngpus > 1): one distributed
  // rank plan per device, connected with plain peer pointers; every call fans out
  std::vector<chol_plan_s*> subs;
};
static bool is_multi(const chol_plan_s* p) { return p && !p->subs.empty(); }
static void invalidate_factor(chol_plan_s* p);

#define CUDA_TRY(x)                                   \
  do {                                                \
    cudaError_t e_ = (x);                             \
    if (e_ != cudaSuccess) return -100 - (int)e_;     \
  } while (0)

// ------------------------------------------------------------------ TMA map
typedef CUresult (*PFN_encodeTiled_t)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*,
                                      const cuuint64_t*, const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave,
                                      CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

// 3-D map over `count` row-major d x d FP64 blocks, box {16, bs, 1}, 128-byte swizzle
static int encode_blocks_map(CUtensorMap* map, double* base, int64_t d, int64_t count, int bs) {
  void* fn = nullptr;
  cudaDriverEntryPointQueryResult q;
  CUDA_TRY(cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fn, cudaEnableDefault, &q));
  if (!fn || q != cudaDriverEntryPointSuccess) return -100 - (int)cudaErrorNotSupported;
  auto encode = reinterpret_cast<PFN_encodeTiled_t>(fn);
  const cuuint64_t dims[3] = {(cuuint64_t)d, (cuuint64_t)d, (cuuint64_t)count};
  const cuuint64_t strides[2] = {(cuuint64_t)d * 8, (cuuint64_t)d * d * 8};
  const cuuint32_t box[3] = {16, (cuuint32_t)bs, 1};
  const cuuint32_t estr[3] = {1, 1, 1};
  CUresult r = encode(map, CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 3, base, dims, strides, box, estr,
                      CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_128B, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                      CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  if (r != CUDA_SUCCESS) return -100 - (int)cudaErrorInvalidValue;
  return 0;
}
static int encode_tile_map(chol_plan_s* p) { return encode_blocks_map(&p->map, p->tiles, p->nb, p->ntiles, p->bs); }

// Dinv workspace of the inverse-form TRSM row slabs (sched.cu J_INV / J_TRSM): N * nb/bs
// blocks of bs x bs (35 MB at n = 46080), and its map
static int make_dinv(chol_plan_s* p) {
  const int64_t nblk = p->N * (p->nb / p->bs);
  cudaError_t e = cudaMalloc(&p->d_dinv, (size_t)nblk * p->bs * p->bs * sizeof(double));
  if (e == cudaErrorMemoryAllocation) {
    cudaGetLastError();
    return -9;
  }
  if (e) return -100 - (int)e;
  return encode_blocks_map(&p->dmap, p->d_dinv, p->bs, nblk, p->bs);
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
    case -10: return "no successful factorization in the plan";
    case -11: return "scheduler made no progress within CHOL_WATCHDOG_S seconds (run aborted)";
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
  if (is_multi(p)) {
    for (chol_plan_s* sp : p->subs) chol_destroy(sp);
    delete p;
    return 0;
  }
  if (p->host) host_trsm_destroy(p->host);
  if (p->sched) sched_destroy(p->sched);
  cudaSetDevice(p->device);
  sched_phase_dump();
  if (p->stream) cudaStreamSynchronize(p->stream);
  for (void* ptr : p->ipc_opened) cudaIpcCloseMemHandle(ptr);
  cudaFree(p->d_inv);
  cudaFree(p->d_rhs);
  cudaFree(p->d_solve_ctl);
  if (p->ev4) cudaEventDestroy(p->ev4);
  if (p->ev5) cudaEventDestroy(p->ev5);
  cudaFree(p->d_slot_map);
  cudaFree(p->d_owner_slot);
  cudaFree(p->d_owned_tile);
  cudaFree(p->d_diag_slots);
  cudaFree(p->d_flags);
  cudaFree(p->d_peer_slots);
  cudaFree(p->d_peer_flags);
  cudaFree(p->d_in_flags);
  cudaFree(p->d_host_flags);
  if (p->h_out_flags) cudaFreeHost(p->h_out_flags);
  if (p->h_epoch) cudaFreeHost(p->h_epoch);
  if (p->s_in) cudaStreamDestroy(p->s_in);
  if (p->s_out) cudaStreamDestroy(p->s_out);
  cudaFree(p->tiles);
  cudaFree(p->d_dinv);
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

static int plan_multi(int64_t n, int64_t nb, int ngpus, const chol_opts_t& opts, chol_plan_t* out);

extern "C" int chol_plan_ex(int64_t n, int64_t nb, int ngpus, const chol_opts_t* o, chol_plan_t* out) {
  if (!out) return -4;
  *out = nullptr;
  if (n <= 0) return -1;
  if (nb <= 0 || n % nb != 0 || nb % 32 != 0) return -2;
  chol_opts_t opts{};
  if (o) opts = *o;
  if (opts.policy < 0 || opts.policy > 2 || opts.executor < 0 || opts.executor > 1 || opts.trsm_pin_distance < 0 ||
      opts.latency_workers < 0 || opts.workers < 0 || opts.grid_p < 0 || opts.grid_q < 0 || opts.trace < 0 ||
      opts.trace > 2 || opts.cpu_trsm_distance < 0 || opts.cpu_threads < 0)
    return -6;
  if (opts.cpu_trsm_distance > 0 && (ngpus != 1 || opts.executor != CHOL_EXEC_SCHEDULER)) return -6;
  int ndev = 0;
  if (cudaGetDeviceCount(&ndev) != cudaSuccess) {
    cudaGetLastError();
    ndev = 0;
  }
  // development check on a one-GPU box: CHOL_MULTI_ONE_DEVICE=1 puts every rank of a
  // multi-device plan on the current device (SMs / ngpus workers each)
  const char* e1d = getenv("CHOL_MULTI_ONE_DEVICE");
  const bool one_dev = e1d && e1d[0] == '1' && ndev >= 1;
  if (ngpus < 1 || (ngpus > ndev && !one_dev)) return -3;
  if (opts.grid_p == 0 && opts.grid_q == 0) {
    opts.grid_p = 1;  // p <= q, as square as possible
    for (int c = 1; c * c <= ngpus; ++c)
      if (ngpus % c == 0) opts.grid_p = c;
    opts.grid_q = ngpus / opts.grid_p;
  }
  if (opts.grid_p * opts.grid_q != ngpus) return -3;
  if (ngpus > 1) return plan_multi(n, nb, ngpus, opts, out);

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
  if ((st = make_dinv(p))) return fail(st);
  if ((e = prepare_kernels(p->bs))) return fail(-100 - (int)e);
  if (opts.executor == CHOL_EXEC_SCHEDULER) {
    if ((st = sched_create(&p->sched, p->N, p->nb, p->bs, p->sms, &p->opts, p->stream))) return fail(st);
    sched_set_dinv(p->sched, p->d_dinv, p->dmap);
    // arrival flags (device), publish flags (host-mapped, polled by chol_factor), copy streams
    if ((e = cudaMalloc(&p->d_in_flags, p->ntiles * sizeof(int))) ||
        (e = cudaHostAlloc(&p->h_out_flags, 2 * p->ntiles * sizeof(int), cudaHostAllocMapped)) ||
        (e = cudaHostGetDevicePointer(&p->d_out_flags, p->h_out_flags, 0)) ||
        (e = cudaHostAlloc(&p->h_epoch, sizeof(int), cudaHostAllocDefault)) ||
        (e = cudaMalloc(&p->d_host_flags, p->ntiles * sizeof(int))) ||
        (e = cudaMalloc(&p->d_peer_flags, 2 * sizeof(int*))) ||
        (e = cudaStreamCreateWithFlags(&p->s_in, cudaStreamNonBlocking)) ||
        (e = cudaStreamCreateWithFlags(&p->s_out, cudaStreamNonBlocking)))
      return fail(-100 - (int)e);
    memset(p->h_out_flags, 0, 2 * p->ntiles * sizeof(int));
    cudaMemset(p->d_in_flags, 0, p->ntiles * sizeof(int));
    cudaMemset(p->d_host_flags, 0, p->ntiles * sizeof(int));
    int* watched[2] = {p->d_in_flags, p->d_host_flags};  // watch owner 0: input arrival, 1: host class
    cudaMemcpy(p->d_peer_flags, watched, 2 * sizeof(int*), cudaMemcpyHostToDevice);
    sched_set_dist(p->sched, nullptr, nullptr, nullptr, p->d_peer_flags, p->d_out_flags);
    if (!sched_host_tasks(p->sched).empty() &&
        (st = host_trsm_create(&p->host, p->device, (int)nb, p->bs, opts.cpu_threads, p->ntiles, p->tiles, p->d_dinv,
                               p->d_host_flags, p->h_out_flags + p->ntiles, sched_host_tasks(p->sched))))
      return fail(st);
  }
  *out = p;
  return 0;
}

extern "C" int chol_plan(int64_t n, int64_t nb, int ngpus, chol_plan_t* out) {
  return chol_plan_ex(n, nb, ngpus, nullptr, out);
}

// ------------------------------------------------------------------ multi-GPU plan
// One process (or one logical rank) per GPU; 2D block-cyclic owner-computes.
extern "C" int chol_plan_dist(int64_t n, int64_t nb, int nranks, int rank, const chol_opts_t* o, chol_plan_t* out) {
  if (!out) return -4;
  *out = nullptr;
  if (n <= 0) return -1;
  if (nb <= 0 || n % nb != 0 || nb % 32 != 0) return -2;
  if (nranks < 1 || rank < 0 || rank >= nranks) return -3;
  chol_opts_t opts{};
  if (o) opts = *o;
  if (opts.policy < 0 || opts.policy > 2 || opts.executor != CHOL_EXEC_SCHEDULER || opts.trsm_pin_distance < 0 ||
      opts.latency_workers < 0 || opts.workers < 0 || opts.grid_p < 0 || opts.grid_q < 0 || opts.trace < 0 ||
      opts.trace > 2 || opts.cpu_trsm_distance != 0 || opts.cpu_threads < 0)  // host class: single GPU only
    return -6;
  if (opts.grid_p == 0 && opts.grid_q == 0) {
    opts.grid_p = 1;
    opts.grid_q = nranks;
  }
  if (opts.grid_p * opts.grid_q != nranks) return -3;
  int ndev = 0;
  if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev < 1) {
    cudaGetLastError();
    return -3;
  }
  auto* p = new (std::nothrow) chol_plan_s();
  if (!p) return -9;
  auto fail = [&](int s) {
    chol_destroy(p);
    return s;
  };
  p->n = n;
  p->nb = nb;
  p->N = n / nb;
  p->ntasks = n_tasks(p->N);
  p->bs = pick_block(nb);
  p->opts = opts;
  p->dist = true;
  p->rank = rank;
  p->nranks = nranks;
  p->p = opts.grid_p;
  p->q = opts.grid_q;
  cudaError_t e;
  if ((e = cudaGetDevice(&p->device))) return fail(-100 - (int)e);
  cudaDeviceGetAttribute(&p->sms, cudaDevAttrMultiProcessorCount, p->device);
  int nowned = 0, ncached = 0;
  dist_layout(p->N, p->p, p->q, rank, p->h_slot_map, &nowned, &ncached);
  p->nowned = nowned;
  p->nslots = nowned + ncached;
  p->ntiles = std::max<int64_t>(p->nslots, 1);
  p->h_owned_tile.assign(nowned, 0);
  std::vector<int> diag;
  for (int64_t t = 0; t < (int64_t)p->h_slot_map.size(); ++t)
    if (p->h_slot_map[t] >= 0 && p->h_slot_map[t] < nowned) p->h_owned_tile[p->h_slot_map[t]] = (int)t;
  for (int64_t k = 0; k < p->N; ++k)
    if (tile_owner_h(k, k, p->p, p->q) == rank) diag.push_back(p->h_slot_map[tile_index(k, k)]);
  p->ndiag = (int)diag.size();
  std::vector<int> oslot;
  owner_slots(p->N, p->p, p->q, oslot);
  const size_t tiles_n = p->h_slot_map.size();
  e = cudaMalloc(&p->tiles, (size_t)p->ntiles * nb * nb * sizeof(double));
  if (e == cudaErrorMemoryAllocation) {
    cudaGetLastError();
    return fail(-9);
  }
  if (e) return fail(-100 - (int)e);
  if ((e = cudaMalloc(&p->d_slot_map, tiles_n * 4)) || (e = cudaMalloc(&p->d_owner_slot, tiles_n * 4)) ||
      (e = cudaMalloc(&p->d_owned_tile, std::max<size_t>(nowned, 1) * 4)) ||
      (e = cudaMalloc(&p->d_diag_slots, std::max<size_t>(diag.size(), 1) * 4)) ||
      (e = cudaMalloc(&p->d_flags, tiles_n * 4)) || (e = cudaMalloc(&p->d_peer_slots, nranks * sizeof(double*))) ||
      (e = cudaMalloc(&p->d_peer_flags, nranks * sizeof(int*))))
    return fail(-100 - (int)e);
  cudaMemcpy(p->d_slot_map, p->h_slot_map.data(), tiles_n * 4, cudaMemcpyHostToDevice);
  cudaMemcpy(p->d_owner_slot, oslot.data(), tiles_n * 4, cudaMemcpyHostToDevice);
  if (nowned) cudaMemcpy(p->d_owned_tile, p->h_owned_tile.data(), nowned * 4, cudaMemcpyHostToDevice);
  if (!diag.empty()) cudaMemcpy(p->d_diag_slots, diag.data(), diag.size() * 4, cudaMemcpyHostToDevice);
  cudaMemset(p->d_flags, 0, tiles_n * 4);
  if ((e = cudaStreamCreateWithFlags(&p->stream, cudaStreamNonBlocking))) return fail(-100 - (int)e);
  if ((e = cudaMalloc(&p->d_info, sizeof(int)))) return fail(-100 - (int)e);
  if ((e = cudaMalloc(&p->d_base, sizeof(uint64_t)))) return fail(-100 - (int)e);
  if (opts.trace) {
    if ((e = cudaMalloc(&p->d_t0, p->ntasks * sizeof(uint64_t)))) return fail(-100 - (int)e);
    if ((e = cudaMalloc(&p->d_t1, p->ntasks * sizeof(uint64_t)))) return fail(-100 - (int)e);
  }
  for (cudaEvent_t* ev : {&p->ev0, &p->ev1, &p->ev2, &p->ev3})
    if ((e = cudaEventCreate(ev))) return fail(-100 - (int)e);
  int st = 0;
  if ((st = encode_tile_map(p))) return fail(st);
  if ((e = prepare_kernels(p->bs))) return fail(-100 - (int)e);
  DistInfo di{p->p, p->q, rank, nranks, p->h_slot_map.data()};
  if ((st = sched_create(&p->sched, p->N, p->nb, p->bs, p->sms, &p->opts, p->stream, &di))) return fail(st);
  if ((st = make_dinv(p))) return fail(st);
  sched_set_dinv(p->sched, p->d_dinv, p->dmap);
  *out = p;
  return 0;
}

namespace {
struct ExportBlob {  // what a rank tells the others (chol_dist_export / chol_dist_connect)
  uint32_t magic, version;
  int32_t pid, device, rank, nranks;
  uint64_t slots_ptr, flags_ptr;
  cudaIpcMemHandle_t slots_h, flags_h;
};
constexpr uint32_t kBlobMagic = 0x43484f4cu;  // "CHOL"
}  // namespace

extern "C" int chol_dist_export(chol_plan_t p, void* blob, int64_t cap, int64_t* len) {
  if (!p || !p->dist) return -4;
  if (len) *len = (int64_t)sizeof(ExportBlob);
  if (!blob) return 0;
  if (cap < (int64_t)sizeof(ExportBlob)) return -4;
  cudaSetDevice(p->device);
  ExportBlob b{};
  b.magic = kBlobMagic;
  b.version = 1;
  b.pid = (int32_t)getpid();
  b.device = p->device;
  b.rank = p->rank;
  b.nranks = p->nranks;
  b.slots_ptr = (uint64_t)(uintptr_t)p->tiles;
  b.flags_ptr = (uint64_t)(uintptr_t)p->d_flags;
  CUDA_TRY(cudaIpcGetMemHandle(&b.slots_h, p->tiles));
  CUDA_TRY(cudaIpcGetMemHandle(&b.flags_h, p->d_flags));
  memcpy(blob, &b, sizeof(b));
  return 0;
}

extern "C" int chol_dist_connect(chol_plan_t p, const void* blobs, int64_t stride) {
  if (!p || !p->dist || !blobs || stride < (int64_t)sizeof(ExportBlob)) return -4;
  if (p->connected) return 0;
  cudaSetDevice(p->device);
  std::vector<double*> slots(p->nranks);
  std::vector<int*> flags(p->nranks);
  const int me = (int)getpid();
  for (int r = 0; r < p->nranks; ++r) {
    ExportBlob b;
    memcpy(&b, static_cast<const char*>(blobs) + r * stride, sizeof(b));
    if (b.magic != kBlobMagic || b.rank != r || b.nranks != p->nranks) return -6;
    if (r == p->rank) {
      slots[r] = p->tiles;
      flags[r] = p->d_flags;
    } else if (b.pid == me) {  // logical ranks in one process: plain device pointers
      if (b.device != p->device) {
        cudaError_t e = cudaDeviceEnablePeerAccess(b.device, 0);
        if (e != cudaSuccess && e != cudaErrorPeerAccessAlreadyEnabled) return -100 - (int)e;
        cudaGetLastError();
      }
      slots[r] = reinterpret_cast<double*>(b.slots_ptr);
      flags[r] = reinterpret_cast<int*>(b.flags_ptr);
    } else {  // another process: map its allocations (NVLink peer memory)
      void *ps = nullptr, *pf = nullptr;
      CUDA_TRY(cudaIpcOpenMemHandle(&ps, b.slots_h, cudaIpcMemLazyEnablePeerAccess));
      p->ipc_opened.push_back(ps);
      CUDA_TRY(cudaIpcOpenMemHandle(&pf, b.flags_h, cudaIpcMemLazyEnablePeerAccess));
      p->ipc_opened.push_back(pf);
      slots[r] = static_cast<double*>(ps);
      flags[r] = static_cast<int*>(pf);
    }
  }
  CUDA_TRY(cudaMemcpy(p->d_peer_slots, slots.data(), p->nranks * sizeof(double*), cudaMemcpyHostToDevice));
  CUDA_TRY(cudaMemcpy(p->d_peer_flags, flags.data(), p->nranks * sizeof(int*), cudaMemcpyHostToDevice));
  sched_set_dist(p->sched, p->d_slot_map, p->d_owner_slot, p->d_peer_slots, p->d_peer_flags, p->d_flags);
  p->connected = true;
  return 0;
}

extern "C" int chol_get_dist(chol_plan_t p, int* rank, int* nranks, int* grid_p, int* grid_q, int64_t* nowned,
                             int64_t* nslots) {
  if (!p) return -4;
  if (rank) *rank = p->rank;
  if (nranks) *nranks = p->nranks;
  if (grid_p) *grid_p = p->p;
  if (grid_q) *grid_q = p->q;
  if (nowned) *nowned = p->dist ? p->nowned : p->ntiles;
  if (nslots) *nslots = p->dist ? p->nslots : p->ntiles;
  return 0;
}

// ------------------------------------------------------------------ one process, ngpus devices
// chol_plan(n, nb, ngpus > 1) (SURVEY §8b process model): rank r of the 2D block-cyclic
// plan (chol_plan_dist) lives on device r; the ranks are connected in-process (plain
// device pointers, cudaDeviceEnablePeerAccess -- NVLink peer memory), and every call
// below fans out to them.  A, L may be host pointers or device pointers (UVA copies).
static int factor_launch(chol_plan_s* p);
static int finish_info(chol_plan_s* p, int* info);

static int plan_multi(int64_t n, int64_t nb, int ngpus, const chol_opts_t& opts, chol_plan_t* out) {
  int dev0 = 0, ndev = 0;
  CUDA_TRY(cudaGetDevice(&dev0));
  CUDA_TRY(cudaGetDeviceCount(&ndev));
  const char* e1d = getenv("CHOL_MULTI_ONE_DEVICE");
  const bool one_dev = e1d && e1d[0] == '1';
  auto* m = new (std::nothrow) chol_plan_s();
  if (!m) return -9;
  m->n = n;
  m->nb = nb;
  m->N = n / nb;
  m->ntiles = m->N * (m->N + 1) / 2;
  m->ntasks = n_tasks(m->N);
  m->bs = pick_block(nb);
  m->opts = opts;
  m->ngpus = m->nranks = ngpus;
  m->device = dev0;
  m->p = opts.grid_p;
  m->q = opts.grid_q;
  chol_opts_t so = opts;
  if (one_dev && so.workers == 0) {
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev0);
    so.workers = std::max(1, sms / ngpus);
  }
  auto fail = [&](int st) {
    cudaSetDevice(dev0);
    if (m->subs.empty())
      delete m;
    else
      chol_destroy(m);
    return st;
  };
  for (int r = 0; r < ngpus; ++r) {
    if (cudaSetDevice(one_dev ? dev0 : r % ndev)) return fail(-3);
    chol_plan_t sp = nullptr;
    const int st = chol_plan_dist(n, nb, ngpus, r, &so, &sp);
    if (st) return fail(st);
    m->subs.push_back(sp);
  }
  constexpr int64_t kStride = 4096;
  const size_t nr = ngpus > 0 ? (size_t)ngpus : 1;
  std::vector<char> blobs(nr * (size_t)kStride, 0);
  for (int r = 0; r < ngpus; ++r) {
    int64_t len = 0;
    int st = chol_dist_export(m->subs[r], nullptr, 0, &len);
    if (st || len > kStride) return fail(st ? st : -8);
    if ((st = chol_dist_export(m->subs[r], blobs.data() + r * kStride, kStride, &len))) return fail(st);
  }
  for (int r = 0; r < ngpus; ++r) {
    const int st = chol_dist_connect(m->subs[r], blobs.data(), kStride);
    if (st) return fail(st);
  }
  cudaSetDevice(dev0);
  *out = m;
  return 0;
}

static int multi_launch(chol_plan_s* m) {
  invalidate_factor(m);
  for (chol_plan_s* sp : m->subs) {
    cudaSetDevice(sp->device);
    const int st = factor_launch(sp);
    if (st) return st;
  }
  return 0;
}
// On the first failing rank the others are aborted (they would spin on its publish flags
// forever), every rank is still waited for, and the first error is returned.
static int multi_finish(chol_plan_s* m, int* info) {
  int best = 0, launches = 0, first_err = 0;
  double t = 0.0;
  for (chol_plan_s* sp : m->subs) {
    cudaSetDevice(sp->device);
    int i = 0;
    const int st = finish_info(sp, &i);
    if (st) {
      if (!first_err) {
        first_err = st;
        for (chol_plan_s* o : m->subs)
          if (o != sp && o->sched) {
            cudaSetDevice(o->device);
            sched_abort(o->sched);
          }
      }
      continue;
    }
    if (i && (!best || i < best)) best = i;
    t = std::max(t, sp->last_factor_s);
    launches += sp->last_launches;
  }
  cudaSetDevice(m->device);
  if (first_err) return first_err;
  m->last_factor_s = t;
  m->last_launches = launches;
  m->factored = true;
  m->last_info = best;
  if (info) *info = best;
  return 0;
}

extern "C" int chol_get_stream(chol_plan_t p, void** stream) {
  if (!p || !stream) return -4;
  if (is_multi(p)) p = p->subs[0];
  *stream = (void*)p->stream;
  return 0;
}

extern "C" int chol_get_info(chol_plan_t p, int64_t* n, int64_t* nb, int* block, int* workers, int* policy,
                             int* executor) {
  if (!p) return -4;
  if (n) *n = p->n;
  if (nb) *nb = p->nb;
  if (block) *block = p->bs;
  if (workers) {
    *workers = p->sched ? sched_workers(p->sched) : 0;
    for (chol_plan_s* sp : p->subs) *workers += sp->sched ? sched_workers(sp->sched) : 0;
  }
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

static int64_t store_slot(const chol_plan_s* p, int64_t i, int64_t j) {
  return p->dist ? p->h_slot_map[tile_index(i, j)] : tile_index(i, j);
}
static bool owns(const chol_plan_s* p, int64_t i, int64_t j) {
  return !p->dist || tile_owner_h(i, j, p->p, p->q) == p->rank;
}

static int scatter_impl(chol_plan_s* p, const double* A, int64_t lda) {
  const int64_t nb = p->nb;
  for (int64_t i = 0; i < p->N; ++i)
    for (int64_t j = 0; j <= i; ++j) {
      if (!owns(p, i, j)) continue;
      double* dst = p->tiles + store_slot(p, i, j) * nb * nb;
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

// Multi-GPU plans write only the tiles this rank owns; rank 0 also zeroes the strictly
// upper tiles (a caller gathering every rank into one buffer gets the full L).
static int gather_impl(chol_plan_s* p, double* L, int64_t ldl) {
  const int64_t nb = p->nb, n = p->n;
  if (p->dist)
    CUDA_TRY(launch_zero_upper_diag(p->tiles, (int)nb, (int)p->N, p->stream, p->d_diag_slots, p->ndiag));
  else
    CUDA_TRY(launch_zero_upper_diag(p->tiles, (int)nb, (int)p->N, p->stream));
  const bool dev = is_device_ptr(L);
  const bool zero_upper = !p->dist || p->rank == 0;
  for (int64_t i = 0; i < p->N; ++i) {
    for (int64_t j = 0; j <= i; ++j) {
      if (!owns(p, i, j)) continue;
      const double* src = p->tiles + store_slot(p, i, j) * nb * nb;
      double* dst = L + i * nb * ldl + j * nb;
      CUDA_TRY(cudaMemcpy2DAsync(dst, ldl * 8, src, nb * 8, nb * 8, nb, cudaMemcpyDefault, p->stream));
    }
    if (zero_upper && dev && (i + 1) * nb < n)
      CUDA_TRY(cudaMemset2DAsync(L + i * nb * ldl + (i + 1) * nb, ldl * 8, 0, (n - (i + 1) * nb) * 8, nb, p->stream));
  }
  if (zero_upper && !dev) host_zero_upper_tiles(L, ldl, n, nb);
  return 0;
}

extern "C" int chol_scatter(chol_plan_t p, const double* A, int64_t lda) {
  if (!p || !A || (reinterpret_cast<uintptr_t>(A) & 7)) return -4;
  if (lda < p->n) return -5;
  if (is_multi(p)) {  // every rank copies its own tiles at once (one stream per device), then wait
    invalidate_factor(p);
    int st = 0;
    for (chol_plan_s* sp : p->subs) {
      cudaSetDevice(sp->device);
      if (!st) st = scatter_impl(sp, A, lda);
    }
    for (chol_plan_s* sp : p->subs) {
      cudaSetDevice(sp->device);
      const cudaError_t e = cudaStreamSynchronize(sp->stream);
      if (e && !st) st = -100 - (int)e;
    }
    cudaSetDevice(p->device);
    return st;
  }
  cudaSetDevice(p->device);
  invalidate_factor(p);
  int st = scatter_impl(p, A, lda);
  if (st) return st;
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  return 0;
}

extern "C" int chol_gather(chol_plan_t p, double* L, int64_t ldl) {
  if (!p || !L || (reinterpret_cast<uintptr_t>(L) & 7)) return -4;
  if (ldl < p->n) return -5;
  if (is_multi(p)) {  // all ranks at once (one stream per device), then wait
    int st = 0;
    for (chol_plan_s* sp : p->subs) {
      cudaSetDevice(sp->device);
      if (!st) st = gather_impl(sp, L, ldl);
    }
    for (chol_plan_s* sp : p->subs) {
      cudaSetDevice(sp->device);
      const cudaError_t e = cudaStreamSynchronize(sp->stream);
      if (e && !st) st = -100 - (int)e;
    }
    cudaSetDevice(p->device);
    return st;
  }
  cudaSetDevice(p->device);
  int st = gather_impl(p, L, ldl);
  if (st) return st;
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  return 0;
}

// The owned tiles occupy slots 0 .. nowned-1 in tile order (dist_layout; identity on
// one GPU): one contiguous copy each way.
static int owned_tiles_copy(chol_plan_t p, void* dst, const void* src, int64_t count) {
  if (!p || !dst || !src || (reinterpret_cast<uintptr_t>(dst) & 7) || (reinterpret_cast<uintptr_t>(src) & 7))
    return -4;
  if (count != (p->dist ? p->nowned : p->ntiles)) return -6;
  cudaSetDevice(p->device);
  CUDA_TRY(cudaMemcpyAsync(dst, src, (size_t)count * p->nb * p->nb * sizeof(double), cudaMemcpyDefault, p->stream));
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  return 0;
}
extern "C" int chol_scatter_tiles(chol_plan_t p, const double* tiles, int64_t count) {
  if (is_multi(p)) return -8;  // per-rank call: use the rank plans (chol_plan_dist)
  if (p) invalidate_factor(p);
  return p ? owned_tiles_copy(p, p->tiles, tiles, count) : -4;
}
extern "C" int chol_gather_tiles(chol_plan_t p, double* tiles, int64_t count) {
  if (is_multi(p)) return -8;
  return p ? owned_tiles_copy(p, tiles, p->tiles, count) : -4;
}

extern "C" int chol_generate(chol_plan_t p, uint64_t seed, int family) {
  if (!p) return -4;
  if (family < 0 || family > 1) return -6;
  invalidate_factor(p);
  if (is_multi(p)) {  // every rank generates its owned tiles at once, then wait
    int st = 0;
    for (chol_plan_s* sp : p->subs) {
      cudaSetDevice(sp->device);
      if (st) break;
      const cudaError_t e = launch_generate(sp->tiles, sp->n, (int)sp->nb, (int)sp->N, seed, family, sp->stream,
                                            sp->d_owned_tile, sp->nowned);
      if (e) st = -100 - (int)e;
    }
    for (chol_plan_s* sp : p->subs) {
      cudaSetDevice(sp->device);
      const cudaError_t e = cudaStreamSynchronize(sp->stream);
      if (e && !st) st = -100 - (int)e;
    }
    cudaSetDevice(p->device);
    return st;
  }
  cudaSetDevice(p->device);
  CUDA_TRY(launch_generate(p->tiles, p->n, (int)p->nb, (int)p->N, seed, family, p->stream,
                           p->dist ? p->d_owned_tile : nullptr, p->nowned));
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
  sp.dinv = p->d_dinv;
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
    CUDA_TRY(launch_trsm(p->bs, p->map, p->dmap, sp, N - 1 - k, p->stream, nlaunch));
    const int m = N - 1 - k;
    sp.mode = 0;
    CUDA_TRY(launch_update(p->bs, p->map, sp, m * (m + 1) / 2, p->stream, nlaunch));
  }
  return 0;
}

// Every call that writes the tile store first forgets the previous factor: chol_solve
// then refuses (-10) until a factorization completes with info = 0, and the cached
// diagonal-block inverses are recomputed (a failed, aborted or overwritten factor is
// never used).
static void invalidate_factor(chol_plan_s* p) {
  p->factored = false;
  p->last_info = -1;
  p->inv_valid = false;
  for (chol_plan_s* sp : p->subs) invalidate_factor(sp);
}

static int factor_launch(chol_plan_s* p) {
  invalidate_factor(p);
  CUDA_TRY(launch_init_info(p->d_info, p->stream));
  if (p->opts.trace) {
    CUDA_TRY(cudaMemsetAsync(p->d_t0, 0xff, p->ntasks * sizeof(uint64_t), p->stream));
    CUDA_TRY(cudaMemsetAsync(p->d_t1, 0, p->ntasks * sizeof(uint64_t), p->stream));
  }
  CUDA_TRY(launch_stamp(p->d_base, p->stream));
  int nl = 0;
  CUDA_TRY(cudaEventRecord(p->ev0, p->stream));
  int st = 0;
  if (p->dist && !p->connected) return -8;
  ++p->epoch;
  if (!p->dist && p->sched && !p->streamed_run)  // input already resident: every tile has arrived
    CUDA_TRY(launch_fill_flags(p->d_in_flags, p->ntiles, (int)p->epoch, p->stream));
  if (p->opts.executor == CHOL_EXEC_HOST)
    st = run_host_sequenced(p, &nl);
  else
    st = sched_run(p->sched, p->map, base_params(p), p->stream, &nl, p->epoch);
  if (st) return st;
  if (p->host) host_trsm_start(p->host, p->epoch);  // the host class follows the kernel's flags
  CUDA_TRY(cudaEventRecord(p->ev1, p->stream));
  p->last_launches = nl;
  return 0;
}

// Host watchdog over the persistent scheduler (wait_plan, factor_streamed): it reads the
// device's completed-node counter every 0.25 s; no progress for CHOL_WATCHDOG_S seconds
// (default 60, 0 = off) aborts the run (sched_abort: the scheduler warps stop handing out
// jobs, the kernel exits) and reports -11 -- a stalled scheduler (a rank that never
// launched, a lost peer flag) is reported instead of hanging the caller.
namespace {
struct Watchdog {
  using clk = std::chrono::steady_clock;
  chol_plan_s* p;
  double limit = 60.0;
  const int* prog = nullptr;
  cudaStream_t ws = nullptr;
  int* h = nullptr;
  int last = -1;
  clk::time_point t_prog = clk::now(), t_check = clk::now();
  explicit Watchdog(chol_plan_s* plan) : p(plan) {
    const char* ew = getenv("CHOL_WATCHDOG_S");
    if (ew) limit = atof(ew);
    prog = p->sched ? sched_progress(p->sched) : nullptr;
    if (prog && limit > 0 &&
        (cudaStreamCreateWithFlags(&ws, cudaStreamNonBlocking) || cudaHostAlloc(&h, sizeof(int), 0))) {
      cudaGetLastError();
      prog = nullptr;  // no watchdog: plain waits
    }
  }
  ~Watchdog() {
    if (ws) cudaStreamDestroy(ws);
    if (h) cudaFreeHost(h);
  }
  bool enabled() const { return prog && limit > 0; }
  // 0 while the scheduler makes progress (or between checks); -11 once a stalled run was aborted
  int check() {
    if (!enabled()) return 0;
    const auto now = clk::now();
    if (std::chrono::duration<double>(now - t_check).count() < 0.25) return 0;
    t_check = now;
    cudaMemcpyAsync(h, prog, sizeof(int), cudaMemcpyDeviceToHost, ws);
    cudaStreamSynchronize(ws);
    if (*h != last) {
      last = *h;
      t_prog = now;
      return 0;
    }
    if (std::chrono::duration<double>(now - t_prog).count() <= limit) return 0;
    sched_abort(p->sched);  // the kernel drains its running jobs and exits
    cudaStreamSynchronize(p->stream);
    cudaGetLastError();
    return -11;
  }
};
}  // namespace

// Wait for the plan's stream under the watchdog.
static int wait_plan(chol_plan_s* p) {
  Watchdog wd(p);
  if (!wd.enabled()) {
    CUDA_TRY(cudaStreamSynchronize(p->stream));
    return 0;
  }
  while (true) {
    const cudaError_t q = cudaStreamQuery(p->stream);
    if (q == cudaSuccess) return 0;
    if (q != cudaErrorNotReady) return -100 - (int)q;
    if (const int w = wd.check()) return w;
    std::this_thread::yield();
  }
}

static int finish_info(chol_plan_s* p, int* info) {
  int h = 0;
  if (const int w = wait_plan(p)) {
    if (p->host) host_trsm_finish(p->host, true);
    return w;
  }
  if (p->host)
    if (const int hs = host_trsm_finish(p->host, false)) return hs;
  CUDA_TRY(cudaMemcpyAsync(&h, p->d_info, sizeof(int), cudaMemcpyDeviceToHost, p->stream));
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  float ms = 0.f;
  CUDA_TRY(cudaEventElapsedTime(&ms, p->ev0, p->ev1));
  p->last_factor_s = ms * 1e-3;
  p->factored = true;
  p->last_info = (h == INT_MAX) ? 0 : h;
  p->inv_valid = false;  // a new factor: the diagonal-block inverses are stale
  if (info) *info = p->last_info;
  return 0;
}

extern "C" int chol_factor_async(chol_plan_t p) {
  if (!p) return -4;
  if (is_multi(p)) return multi_launch(p);
  cudaSetDevice(p->device);
  return factor_launch(p);
}

extern "C" int chol_wait(chol_plan_t p, int* info) {
  if (!p) return -4;
  if (is_multi(p)) return multi_finish(p, info);
  cudaSetDevice(p->device);
  return finish_info(p, info);
}

extern "C" int chol_factor_inplace(chol_plan_t p, int* info) {
  if (!p) return -4;
  if (is_multi(p)) {
    const int st = multi_launch(p);
    return st ? st : multi_finish(p, info);
  }
  cudaSetDevice(p->device);
  int st = factor_launch(p);
  if (st) return st;
  return finish_info(p, info);
}

// chol_factor from HOST memory with the persistent scheduler: the factorization starts
// on the first tile while the rest is still being copied in (per-tile arrival flags
// gate each tile's first task), and every off-diagonal L tile is copied out as soon as
// its TRSM publishes it; only the diagonal tiles are copied after the kernel ends.
static int factor_streamed(chol_plan_s* p, const double* A, int64_t lda, double* L, int64_t ldl, int* info) {
  const int64_t nb = p->nb, N = p->N, n = p->n;
  CUDA_TRY(cudaEventRecord(p->ev2, p->stream));
  p->streamed_run = true;
  const int st = factor_launch(p);  // epoch++, scheduler kernel waits on the arrival flags
  p->streamed_run = false;
  if (st) return st;
  *p->h_epoch = (int)p->epoch;
  CUDA_TRY(cudaStreamWaitEvent(p->s_in, p->ev2, 0));
  CUDA_TRY(cudaStreamWaitEvent(p->s_out, p->ev2, 0));
  // from here on every exit path waits for the copy streams (they read A / write L, the
  // caller's memory) and joins the zeroing thread before returning
  int rc = 0;
  auto copy_in = [&](int64_t i, int64_t j) -> int {
    const int64_t t = tile_index(i, j);
    CUDA_TRY(cudaMemcpy2DAsync(p->tiles + t * nb * nb, nb * 8, A + i * nb * lda + j * nb, lda * 8, nb * 8, nb,
                               cudaMemcpyDefault, p->s_in));
    CUDA_TRY(cudaMemcpyAsync(p->d_in_flags + t, p->h_epoch, sizeof(int), cudaMemcpyHostToDevice, p->s_in));
    return 0;
  };
  // the scheduler's watch order (sched_arrival_order)
  std::vector<std::pair<int, int>> arr;
  sched_arrival_order(p->sched, arr);
  for (size_t a = 0; a < arr.size() && !rc; ++a) rc = copy_in(arr[a].first, arr[a].second);
  if (rc) {  // the kernel waits for arrivals that will never come: stop it
    sched_abort(p->sched);
    cudaStreamSynchronize(p->stream);
    cudaStreamSynchronize(p->s_in);
    cudaGetLastError();
    return rc;
  }
  // L's strictly upper tiles are zeroed on the host once the input has been read:
  // concurrent with the input copies the memset competes with the copy engine for
  // host DRAM bandwidth (measured: arrivals ~2x slower, e2e 90 -> 80 ms at n=19200)
  struct Joiner {
    std::thread t;
    ~Joiner() {
      if (t.joinable()) t.join();
    }
  } zero_upper{std::thread([=] {
    cudaStreamSynchronize(p->s_in);
    host_zero_upper_tiles(L, ldl, n, nb);
  })};
  // stream out every tile as it becomes final: L_kk (the POTRF leaves the strictly
  // upper triangle of diagonal tiles zeroed), then L_ik, in publication order
  std::vector<int64_t> pending;
  for (int64_t k = 0; k < N; ++k)
    for (int64_t i = k; i < N; ++i) pending.push_back(tile_index(i, k));
  std::vector<int> row_of(p->ntiles), col_of(p->ntiles);
  for (int64_t i = 0; i < N; ++i)
    for (int64_t j = 0; j <= i; ++j) {
      row_of[tile_index(i, j)] = (int)i;
      col_of[tile_index(i, j)] = (int)j;
    }
  auto copy_out = [&](int64_t t) {
    const int64_t i = row_of[t], j = col_of[t];
    const cudaError_t e = cudaMemcpy2DAsync(L + i * nb * ldl + j * nb, ldl * 8, p->tiles + t * nb * nb, nb * 8,
                                            nb * 8, nb, cudaMemcpyDefault, p->s_out);
    if (e && !rc) rc = -100 - (int)e;
  };
  Watchdog wd(p);
  const volatile int* outf = p->h_out_flags;
  size_t head = 0;
  while (head < pending.size() && !rc) {
    bool progressed = false;
    for (size_t w = head; w < pending.size() && w < head + 256; ++w) {
      const int64_t t = pending[w];
      if (t < 0 || outf[t] != (int)p->epoch) continue;
      copy_out(t);
      pending[w] = -1;
      progressed = true;
    }
    while (head < pending.size() && pending[head] < 0) ++head;
    if (!progressed) {
      const cudaError_t q = cudaStreamQuery(p->stream);
      if (q == cudaSuccess) {  // kernel done: take the rest
        for (size_t w = head; w < pending.size(); ++w)
          if (pending[w] >= 0) {
            copy_out(pending[w]);
            pending[w] = -1;
          }
        head = pending.size();
      } else if (q != cudaErrorNotReady) {  // a fault: the query fails from now on
        rc = -100 - (int)q;
      } else if (const int w = wd.check()) {  // stalled: aborted, report -11
        rc = w;
      } else {
        std::this_thread::yield();
      }
    }
  }
  int st2 = 0;
  if (!rc) {
    // ev3 after the last output copy: the timed span covers the exposed transfers
    cudaEvent_t out_done;
    cudaError_t e = cudaEventCreateWithFlags(&out_done, cudaEventDisableTiming);
    if (!e) e = cudaEventRecord(out_done, p->s_out);
    if (!e) e = cudaStreamWaitEvent(p->stream, out_done, 0);
    if (out_done) cudaEventDestroy(out_done);
    if (!e) e = cudaEventRecord(p->ev3, p->stream);
    if (e) rc = -100 - (int)e;
    st2 = rc ? 0 : finish_info(p, info);
  }
  const cudaError_t e_in = cudaStreamSynchronize(p->s_in);
  const cudaError_t e_out = cudaStreamSynchronize(p->s_out);
  zero_upper.t.join();
  if (rc) {
    p->factored = false;
    return rc;
  }
  if (st2) return st2;
  if (e_in) return -100 - (int)e_in;
  if (e_out) return -100 - (int)e_out;
  float tot = 0.f;
  CUDA_TRY(cudaEventElapsedTime(&tot, p->ev2, p->ev3));
  p->last_layout_s = tot * 1e-3 - p->last_factor_s;  // exposed (non-overlapped) transfer time
  return 0;
}

extern "C" int chol_factor(chol_plan_t p, const double* A, int64_t lda, double* L, int64_t ldl, int* info) {
  if (!p || !A || !L || (reinterpret_cast<uintptr_t>(A) & 7) || (reinterpret_cast<uintptr_t>(L) & 7)) return -4;
  if (lda < p->n || ldl < p->n) return -5;
  if (is_multi(p)) {  // owners pull their tiles of A, factor together, write their tiles of L
    const auto t0 = std::chrono::steady_clock::now();
    int st = chol_scatter(p, A, lda);
    if (!st) st = chol_factor_inplace(p, info);
    if (!st) st = chol_gather(p, L, ldl);
    const double tot = std::chrono::duration<double>(std::chrono::steady_clock::now() - t0).count();
    p->last_layout_s = tot - p->last_factor_s;
    return st;
  }
  cudaSetDevice(p->device);
  if (!p->dist && p->sched && !is_device_ptr(A) && !is_device_ptr(L)) return factor_streamed(p, A, lda, L, ldl, info);
  CUDA_TRY(cudaEventRecord(p->ev2, p->stream));
  int st = scatter_impl(p, A, lda);
  if (st) return st;
  if ((st = factor_launch(p))) return st;
  if (p->host) {
    // with the host CPU class nothing may wait behind the kernel on p->stream while it runs:
    // copies queued there share the copy engines' hardware queues with the host driver's
    // copies, which the kernel itself waits for (false serialization -> deadlock)
    if ((st = finish_info(p, info))) return st;
    if ((st = gather_impl(p, L, ldl))) return st;
    CUDA_TRY(cudaEventRecord(p->ev3, p->stream));
    CUDA_TRY(cudaStreamSynchronize(p->stream));
  } else {
    if ((st = gather_impl(p, L, ldl))) return st;
    CUDA_TRY(cudaEventRecord(p->ev3, p->stream));
    if ((st = finish_info(p, info))) return st;
  }
  float tot = 0.f;
  CUDA_TRY(cudaEventElapsedTime(&tot, p->ev2, p->ev3));
  p->last_layout_s = tot * 1e-3 - p->last_factor_s;
  return 0;
}

extern "C" int chol_set_task_priorities(chol_plan_t p, const double* prio, int64_t ntasks) {
  if (!p || !prio) return -4;
  if (is_multi(p)) {
    for (chol_plan_s* sp : p->subs)
      if (const int st = chol_set_task_priorities(sp, prio, ntasks)) return st;
    return 0;
  }
  if (!p->sched) return -8;
  cudaSetDevice(p->device);
  CUDA_TRY(cudaStreamSynchronize(p->stream));  // no factorization in flight reads the tables
  return sched_set_priorities(p->sched, prio, ntasks);
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

// ------------------------------------------------------------------ solve
// A X = B with the factor of the last successful factorization (solve.cu): the
// right-hand sides are copied (host or device, any ldb) into a padded device buffer,
// solved by the forward and backward sweeps, and copied back.
extern "C" int chol_solve(chol_plan_t p, double* B, int64_t ldb, int64_t nrhs) {
  if (!p || !B || (reinterpret_cast<uintptr_t>(B) & 7)) return -4;
  if (is_multi(p)) return -8;
  if (nrhs < 1) return -6;
  if (ldb < nrhs) return -5;
  if (p->dist) return -8;
  if (!p->factored || p->last_info != 0) return -10;
  cudaSetDevice(p->device);
  const int64_t n = p->n;
  // columns per work item: 1 (register-streamed matrix-vector sweeps), 32 (DMMA sweeps
  // at block 96 -- also for 2..8 columns: one padded 32-column chunk beats the 8-column
  // SIMT item), 8 or 32 (SIMT sweeps at blocks 64 / 32)
  // 48 at block 96 whenever that takes fewer chunks than 32 (k_sweep_db: both operands
  // double-buffered; a 48-column chunk costs about as much as a 32-column one: n = 19200, nrhs
  // 48 3.03 vs 3.46 ms, 96 3.98 vs 4.54, 192 6.37 vs 7.09 (64-column k_sweep_mma), n = 46080,
  // nrhs 960 152.6 vs 159.4 ms; nrhs 64: 3.94 vs 3.46 -- two chunks either way -- keeps 32;
  // profiles/r02/solve_db_r02s.txt).  CHOL_SOLVE_RC=32 / 48 / 64 forces one (development switch)
  const char* erc = getenv("CHOL_SOLVE_RC");
  const int rc_mma = erc ? (atoi(erc) == 64 ? 64 : atoi(erc) == 48 ? 48 : 32)
                         : ((nrhs + 47) / 48 < (nrhs + 31) / 32 ? 48 : 32);
  const int rc = nrhs == 1 ? 1 : (nrhs <= 8 && p->bs != 96) ? 8 : (p->bs == 96 ? rc_mma : 32);
  const int nchunks = (int)((nrhs + rc - 1) / rc), ldw = rc * nchunks;
  const int64_t nblocks = n / p->bs;
  // one column: + 2 n doubles of chain buffers (forward / backward block results, solve.cu)
  const size_t need = (size_t)n * ldw + (rc == 1 ? 2 * (size_t)n : 0), ctl = 2 + 2 * (size_t)nblocks * nchunks;
  if (!p->d_inv) {
    cudaError_t e = cudaMalloc(&p->d_inv, 3 * (size_t)n * p->bs * sizeof(double));
    if (e) return e == cudaErrorMemoryAllocation ? -9 : -100 - (int)e;
  }
  if (p->rhs_cap < need) {
    cudaFree(p->d_rhs);
    p->d_rhs = nullptr;
    p->rhs_cap = 0;
    cudaError_t e = cudaMalloc(&p->d_rhs, need * sizeof(double));
    if (e) return e == cudaErrorMemoryAllocation ? -9 : -100 - (int)e;
    p->rhs_cap = need;
  }
  if (p->ctl_cap < ctl) {
    cudaFree(p->d_solve_ctl);
    p->d_solve_ctl = nullptr;
    p->ctl_cap = 0;
    cudaError_t e = cudaMalloc(&p->d_solve_ctl, ctl * sizeof(int));
    if (e) return e == cudaErrorMemoryAllocation ? -9 : -100 - (int)e;
    p->ctl_cap = ctl;
  }
  if (!p->ev4) {
    CUDA_TRY(cudaEventCreate(&p->ev4));
    CUDA_TRY(cudaEventCreate(&p->ev5));
  }
  CUDA_TRY(cudaEventRecord(p->ev2, p->stream));
  if (ldw != nrhs) CUDA_TRY(cudaMemsetAsync(p->d_rhs, 0, (size_t)n * ldw * sizeof(double), p->stream));
  CUDA_TRY(cudaMemcpy2DAsync(p->d_rhs, ldw * 8, B, ldb * 8, nrhs * 8, n, cudaMemcpyDefault, p->stream));
  SolveArgs a{};
  a.tiles = p->tiles;
  a.n = n;
  a.nb = (int)p->nb;
  a.sb = p->bs;
  a.inv = p->d_inv;
  a.inv_valid = p->inv_valid;
  a.W = p->d_rhs;
  a.ldw = ldw;
  a.nchunks = nchunks;
  a.rc = rc;
  a.ctl = p->d_solve_ctl;
  a.chain = rc == 1 ? p->d_rhs + (size_t)n * ldw : nullptr;
  a.sms = p->sms;
  // development: CHOL_SOLVE_TRACE=<file> writes per-item sweep timestamps (solve.cu)
  const char* trace_path = getenv("CHOL_SOLVE_TRACE");
  const size_t ntr = 2 * (size_t)nblocks * nchunks * 6;
  if (trace_path) CUDA_TRY(cudaMalloc(&a.trace, ntr * sizeof(uint64_t)));
  int nl = 0;
  CUDA_TRY(cudaEventRecord(p->ev4, p->stream));
  CUDA_TRY(solve_run(a, p->stream, &nl));
  CUDA_TRY(cudaEventRecord(p->ev5, p->stream));
  if (trace_path) {
    std::vector<uint64_t> h(ntr);
    CUDA_TRY(cudaMemcpyAsync(h.data(), a.trace, ntr * sizeof(uint64_t), cudaMemcpyDeviceToHost, p->stream));
    CUDA_TRY(cudaStreamSynchronize(p->stream));
    cudaFree(a.trace);
    if (FILE* f = fopen(trace_path, "wb")) {
      fwrite(h.data(), sizeof(uint64_t), ntr, f);
      fclose(f);
    }
  }
  p->inv_valid = true;
  CUDA_TRY(cudaMemcpy2DAsync(B, ldb * 8, p->d_rhs, ldw * 8, nrhs * 8, n, cudaMemcpyDefault, p->stream));
  CUDA_TRY(cudaEventRecord(p->ev3, p->stream));
  CUDA_TRY(cudaStreamSynchronize(p->stream));
  float ms = 0.f, ms2 = 0.f;
  CUDA_TRY(cudaEventElapsedTime(&ms, p->ev2, p->ev3));
  CUDA_TRY(cudaEventElapsedTime(&ms2, p->ev4, p->ev5));
  p->last_solve_s = ms * 1e-3;
  p->last_sweeps_s = ms2 * 1e-3;
  p->last_launches = nl;
  return 0;
}

extern "C" int chol_last_solve_times(chol_plan_t p, double* total_s, double* sweeps_s) {
  if (!p) return -4;
  if (total_s) *total_s = p->last_solve_s;
  if (sweeps_s) *sweeps_s = p->last_sweeps_s;
  return 0;
}

// ------------------------------------------------------------------ trace
extern "C" int chol_trace(chol_plan_t p, chol_task_rec_t* recs, int64_t cap, int64_t* nrecs, double* makespan_s) {
  if (!p) return -4;
  if (!p->opts.trace || !p->factored) return -7;
  if (is_multi(p)) {
    // every rank records the tasks it ran, relative to its own launch stamp (globaltimer,
    // one clock per device): shift to absolute, merge by task, emit in Algorithm 1 order
    const int64_t N = p->N;
    std::vector<chol_task_rec_t> all(p->ntasks);
    std::vector<char> have(p->ntasks, 0);
    std::vector<chol_task_rec_t> part(p->ntasks);
    uint64_t lo = UINT64_MAX, hi = 0;
    for (chol_plan_s* sp : p->subs) {
      int64_t nr = 0;
      double ms = 0.0;
      int st = chol_trace(sp, part.data(), (int64_t)part.size(), &nr, &ms);
      if (st) return st;
      uint64_t base = 0;
      cudaSetDevice(sp->device);
      CUDA_TRY(cudaMemcpy(&base, sp->d_base, sizeof(base), cudaMemcpyDeviceToHost));
      for (int64_t x = 0; x < nr; ++x) {
        chol_task_rec_t r = part[x];
        r.t0_ns += base;
        r.t1_ns += base;
        const int64_t id = r.type == T_POTRF ? id_potrf(N, r.k)
                           : r.type == T_TRSM ? id_trsm(N, r.i, r.k)
                           : r.type == T_SYRK ? id_syrk(N, r.j, r.k)
                                              : id_gemm(N, r.i, r.j, r.k);
        all[id] = r;
        have[id] = 1;
        lo = std::min(lo, r.t0_ns);
        hi = std::max(hi, r.t1_ns);
      }
    }
    cudaSetDevice(p->device);
    int64_t w = 0;
    auto emit = [&](int64_t id) {
      if (!have[id]) return;
      if (recs && w < cap) {
        recs[w] = all[id];
        recs[w].t0_ns -= lo;
        recs[w].t1_ns -= lo;
      }
      ++w;
    };
    for (int k = 0; k < N; ++k) {
      emit(id_potrf(N, k));
      for (int i = k + 1; i < N; ++i) emit(id_trsm(N, i, k));
      for (int j = k + 1; j < N; ++j) {
        emit(id_syrk(N, j, k));
        for (int i = j + 1; i < N; ++i) emit(id_gemm(N, i, j, k));
      }
    }
    if (nrecs) *nrecs = w;
    if (makespan_s) *makespan_s = (hi > lo) ? (hi - lo) * 1e-9 : 0.0;
    return 0;
  }
  cudaSetDevice(p->device);
  std::vector<uint64_t> t0(p->ntasks), t1(p->ntasks);
  CUDA_TRY(cudaMemcpy(t0.data(), p->d_t0, p->ntasks * 8, cudaMemcpyDeviceToHost));
  CUDA_TRY(cudaMemcpy(t1.data(), p->d_t1, p->ntasks * 8, cudaMemcpyDeviceToHost));
  const int64_t N = p->N;
  uint64_t lo = UINT64_MAX, hi = 0;
  int64_t w = 0;
  auto emit = [&](int type, int i, int j, int k, int64_t id) {
    if (p->dist && t0[id] == UINT64_MAX) return;  // task ran on another rank
    const uint64_t a = t0[id], b = t1[id] >> 16;
    if (t0[id] != UINT64_MAX) {
      lo = std::min(lo, a);
      hi = std::max(hi, b);
    }
    if (recs && w < cap) {
      chol_task_rec_t& r = recs[w];
      r.type = (uint8_t)type;
      r.gpu = (uint8_t)p->rank;
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
  if (is_multi(p)) return -8;
  if (!p->sched || p->opts.trace != 2 || !p->factored) return -7;
  cudaSetDevice(p->device);
  return sched_job_trace(p->sched, out, cap, njobs);  // 5 u64 per job
}

extern "C" int chol_job_desc(chol_plan_t p, int32_t* out, int64_t cap, int64_t* njobs) {
  if (!p) return -4;
  if (is_multi(p)) return -8;
  if (!p->sched) return -7;
  return sched_job_desc(p->sched, out, cap, njobs);
}

// ------------------------------------------------------------------ calibration / single tasks
extern "C" int chol_run_task(chol_plan_t p, int type, int i, int j, int k, int reps, double* ms) {
  if (!p) return -4;
  if (is_multi(p)) return -8;
  if (p->dist) return -8;
  const int N = (int)p->N;
  if (type < 0 || type > 3 || reps < 1 || k < 0 || k >= N) return -6;
  if (type == T_TRSM && !(i > k && i < N)) return -6;
  if (type == T_SYRK && !(j > k && j < N)) return -6;
  if (type == T_GEMM && !(i > j && j > k && i < N)) return -6;
  cudaSetDevice(p->device);
  invalidate_factor(p);
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
      CUDA_TRY(launch_trsm(p->bs, p->map, p->dmap, sp, 1, p->stream, &nl));
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
  if (is_multi(p)) return -8;
  if (p->dist) return -8;
  const int N = (int)p->N;
  if (type < 0 || type > 3 || reps < 1 || count < 1) return -6;
  // instances at step k = 0: POTRF on diagonal tiles 0..count-1, TRSM (i, 0),
  // SYRK (j, 0), GEMM (i, j, 0) -- all with distinct output tiles.
  const int maxc = type == T_POTRF ? N : type == T_GEMM ? (N - 1) * (N - 2) / 2 : N - 1;
  if (count > maxc && !(p->sched && type == T_TRSM)) return -6;  // scheduler: TRSM_i_k over all k
  cudaSetDevice(p->device);
  invalidate_factor(p);
  StepParams sp = base_params(p);
  sp.tr_t0 = sp.tr_t1 = nullptr;
  sp.tr_base = nullptr;
  sp.k = 0;
  CUDA_TRY(launch_init_info(p->d_info, p->stream));
  int nl = 0;
  if (p->sched) {  // the persistent scheduler, the factorization's own executor (reading R9)
    SchedState* bst = nullptr;
    if (const int st = sched_create_batch(&bst, p->N, p->nb, p->bs, p->sms, &p->opts, type, count)) return st;
    sched_set_dinv(bst, p->d_dinv, p->dmap);
    int st = 0;
    for (int r = 0; r <= reps && !st; ++r) {  // r = 0: untimed warm-up
      if (r == 1) CUDA_TRY(cudaEventRecord(p->ev0, p->stream));
      st = sched_run(bst, p->map, sp, p->stream, &nl, ++p->epoch);
    }
    cudaError_t e = cudaEventRecord(p->ev1, p->stream);
    if (!e) e = cudaStreamSynchronize(p->stream);
    sched_destroy(bst);
    if (st) return st;
    if (e) return -100 - (int)e;
    float t = 0.f;
    CUDA_TRY(cudaEventElapsedTime(&t, p->ev0, p->ev1));
    if (ms) *ms = t / reps / count;
    return 0;
  }
  CUDA_TRY(cudaEventRecord(p->ev0, p->stream));
  for (int r = 0; r < reps; ++r) {
    if (type == T_POTRF) {
      CUDA_TRY(launch_potrf(p->bs, p->map, sp, count, p->stream, &nl));
    } else if (type == T_TRSM) {
      sp.i0 = 1;
      CUDA_TRY(launch_trsm(p->bs, p->map, p->dmap, sp, count, p->stream, &nl));
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
