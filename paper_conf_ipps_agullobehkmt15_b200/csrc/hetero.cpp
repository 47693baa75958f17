// Second resource class: host CPU cores (§V-C, L780-823 and
// the static rule actually executed in Fig. 11: every TRSM at least d tiles
// below the diagonal is forced on the CPUs).  The device scheduler turns such a TRSM_i_k
// into two job-less nodes (sched.cu): OUT publishes "inputs final" through a host-mapped
// flag when L_kk, A_ik and the inverses Dinv_k of L_kk's diagonal blocks are ready; IN is
// fired by the watcher once the host has written L_ik back and raised the tile's host flag.
// In between, this driver thread copies the inputs down, solves X <- X L_kk^{-T} on the
// host cores in the same inverse form as the GPU row slabs (R19) -- per column
// block cb of 96: Y = X[:, cb] - X[:, :cb] L[cb, :cb]^T, X[:, cb] = Y Dinv_cb^T -- with an
// AVX-512 dot-product micro-kernel (both operands K-contiguous, no packing), and copies the
// result up.  Host-only code: no kernels.
#include <cuda_runtime.h>

#include <atomic>
#include <cstdio>
#include <cstdlib>
#include <chrono>
#include <condition_variable>
#include <cstring>
#include <functional>
#include <mutex>
#include <thread>
#include <vector>

#include <immintrin.h>

#include "hetero.h"

namespace chol {
namespace {

// C[r][j] (ldc) -= sum_k A[r][k] B[j][k] for r < 4, j < nj (nj <= 6), K % 8 == 0
__attribute__((target("avx512f"))) void mk_4x6_avx512(const double* A, int64_t lda, const double* B, int64_t ldb,
                                                       int K, double* C, int64_t ldc, int nj, double sign) {
  __m512d acc[4][6];
  for (int r = 0; r < 4; ++r)
    for (int j = 0; j < 6; ++j) acc[r][j] = _mm512_setzero_pd();
  for (int k = 0; k < K; k += 8) {
    __m512d a[4], b[6];
    for (int r = 0; r < 4; ++r) a[r] = _mm512_loadu_pd(A + r * lda + k);
    for (int j = 0; j < 6; ++j) b[j] = j < nj ? _mm512_loadu_pd(B + j * ldb + k) : _mm512_setzero_pd();
    for (int r = 0; r < 4; ++r)
      for (int j = 0; j < 6; ++j) acc[r][j] = _mm512_fmadd_pd(a[r], b[j], acc[r][j]);
  }
  for (int r = 0; r < 4; ++r)
    for (int j = 0; j < nj; ++j) C[r * ldc + j] += sign * _mm512_reduce_add_pd(acc[r][j]);
}

void mk_4x6_scalar(const double* A, int64_t lda, const double* B, int64_t ldb, int K, double* C, int64_t ldc, int nj,
                   double sign) {
  for (int r = 0; r < 4; ++r)
    for (int j = 0; j < nj; ++j) {
      double s = 0.0;
      for (int k = 0; k < K; ++k) s += A[r * lda + k] * B[j * ldb + k];
      C[r * ldc + j] += sign * s;
    }
}

const bool kAvx512 = __builtin_cpu_supports("avx512f");

// C (4 x n) += sign * A (4 x K) B^T (B: n x K), row-major, n % 6 handled
void gemm_nt_4rows(const double* A, int64_t lda, const double* B, int64_t ldb, int K, double* C, int64_t ldc, int n,
                   double sign) {
  for (int j0 = 0; j0 < n; j0 += 6) {
    const int nj = n - j0 < 6 ? n - j0 : 6;
    if (kAvx512)
      mk_4x6_avx512(A, lda, B + j0 * ldb, ldb, K, C + j0, ldc, nj, sign);
    else
      mk_4x6_scalar(A, lda, B + j0 * ldb, ldb, K, C + j0, ldc, nj, sign);
  }
}

}  // namespace

// Rows [r0, r0+4) of X (nb x nb, row-major) <- X L^{-T}, inverse form, block bs.
static void trsm_rows(double* X, const double* L, const double* dinv, int nb, int bs, int r0, double* y) {
  const int nbb = nb / bs;
  double* xr = X + (int64_t)r0 * nb;
  for (int cb = 0; cb < nbb; ++cb) {
    // y = X[r, cb] - X[r, :cb] L[cb, :cb]^T   (4 x bs, ld bs)
    for (int r = 0; r < 4; ++r) std::memcpy(y + r * bs, xr + (int64_t)r * nb + cb * bs, bs * sizeof(double));
    if (cb > 0) gemm_nt_4rows(xr, nb, L + (int64_t)cb * bs * nb, nb, cb * bs, y, bs, bs, -1.0);
    // X[r, cb] = y Dinv_cb^T
    double* out = xr + cb * bs;
    for (int r = 0; r < 4; ++r) std::memset(out + (int64_t)r * nb, 0, bs * sizeof(double));
    gemm_nt_4rows(y, bs, dinv + (int64_t)cb * bs * bs, bs, bs, out, nb, bs, 1.0);
  }
}

struct HostTrsm {
  // configuration
  int device = 0;
  int nb = 0, bs = 0, nthreads = 1;
  int64_t ntiles = 0;
  double* tiles = nullptr;         // device tile store
  const double* d_dinv = nullptr;  // device Dinv workspace ([N][nb/bs] bs x bs)
  int* d_host_flags = nullptr;     // device: per tile, epoch in which the host wrote L_ik back
  const volatile int* ready = nullptr;  // host-mapped: per tile, epoch in which OUT published
  std::vector<std::pair<int, int>> tasks;  // (i, k), Algorithm 1 order
  // run state
  std::thread driver;
  std::atomic<bool> stop{false};
  unsigned epoch = 0;
  int status = 0;
  int done_tasks = 0;
  // buffers (pinned)
  double *hX = nullptr, *hL = nullptr, *hD = nullptr;
  int* h_epoch = nullptr;
  cudaStream_t s = nullptr;
  // worker pool for the row loop
  std::vector<std::thread> pool;
  std::mutex mu;
  std::condition_variable cv_go, cv_done;
  int gen = 0, busy = 0;
  bool quit = false;
  std::function<void(int)> job;

  int init() {
    if (cudaStreamCreateWithFlags(&s, cudaStreamNonBlocking)) return -1;
    const size_t tile = (size_t)nb * nb * sizeof(double);
    if (cudaHostAlloc(&hX, tile, 0) || cudaHostAlloc(&hL, tile, 0) ||
        cudaHostAlloc(&hD, (size_t)nb * bs * sizeof(double), 0) || cudaHostAlloc(&h_epoch, sizeof(int), 0))
      return -1;
    for (int w = 1; w < nthreads; ++w)
      pool.emplace_back([this, w] {
        int seen = 0;
        while (true) {
          std::function<void(int)> f;
          {
            std::unique_lock<std::mutex> lk(mu);
            cv_go.wait(lk, [&] { return quit || gen != seen; });
            if (quit) return;
            seen = gen;
            f = job;
          }
          f(w);
          std::lock_guard<std::mutex> lk(mu);
          if (--busy == 0) cv_done.notify_all();
        }
      });
    return 0;
  }
  // run f(thread) on every thread of the pool (the caller is thread 0)
  void parallel(const std::function<void(int)>& f) {
    {
      std::lock_guard<std::mutex> lk(mu);
      job = f;
      busy = nthreads - 1;
      ++gen;
    }
    cv_go.notify_all();
    f(0);
    std::unique_lock<std::mutex> lk(mu);
    cv_done.wait(lk, [&] { return busy == 0; });
  }
  void solve_tile() {
    std::atomic<int> next{0};
    const int nchunks = nb / 4;
    parallel([&](int) {
      std::vector<double> y(4 * (size_t)bs);
      for (int c = next.fetch_add(1); c < nchunks; c = next.fetch_add(1)) trsm_rows(hX, hL, hD, nb, bs, 4 * c, y.data());
    });
  }
  void run() {
    const bool dbg = getenv("CHOL_HOST_DEBUG") != nullptr;  // development: driver progress on stderr
    const size_t tile_elems = (size_t)nb * nb;
    const int nbb = nb / bs;
    int cur_k = -1;
    *h_epoch = (int)epoch;
    for (size_t q = 0; q < tasks.size() && !status; ++q) {
      const int i = tasks[q].first, k = tasks[q].second;
      const int64_t t = (int64_t)i * (i + 1) / 2 + k, tkk = (int64_t)k * (k + 1) / 2 + k;
      if (dbg) fprintf(stderr, "host trsm %zu/%zu (%d,%d): waiting (flag %d, epoch %u)\n", q, tasks.size(), i, k,
                       ready[t], epoch);
      while (ready[t] != (int)epoch) {  // OUT published: L_kk, A_ik and Dinv_k are final
        if (stop.load(std::memory_order_relaxed)) return;
        std::this_thread::yield();
      }
      if (dbg) fprintf(stderr, "host trsm (%d,%d): ready\n", i, k);
      cudaError_t e = cudaSuccess;
      if (k != cur_k) {
        e = cudaMemcpyAsync(hL, tiles + tkk * tile_elems, tile_elems * sizeof(double), cudaMemcpyDeviceToHost, s);
        if (!e)
          e = cudaMemcpyAsync(hD, d_dinv + (size_t)k * nbb * bs * bs, (size_t)nbb * bs * bs * sizeof(double),
                              cudaMemcpyDeviceToHost, s);
        cur_k = k;
      }
      if (!e) e = cudaMemcpyAsync(hX, tiles + t * tile_elems, tile_elems * sizeof(double), cudaMemcpyDeviceToHost, s);
      if (dbg) fprintf(stderr, "host trsm (%d,%d): copies issued (%d)\n", i, k, (int)e);
      if (!e) e = cudaStreamSynchronize(s);
      if (dbg) fprintf(stderr, "host trsm (%d,%d): inputs on host (%d)\n", i, k, (int)e);
      if (e) {
        status = -100 - (int)e;
        return;
      }
      solve_tile();
      if (dbg) fprintf(stderr, "host trsm (%d,%d): solved\n", i, k);
      e = cudaMemcpyAsync(tiles + t * tile_elems, hX, tile_elems * sizeof(double), cudaMemcpyHostToDevice, s);
      if (!e) e = cudaMemcpyAsync(d_host_flags + t, h_epoch, sizeof(int), cudaMemcpyHostToDevice, s);
      if (!e) e = cudaStreamSynchronize(s);  // hX is reused by the next task
      if (e) {
        status = -100 - (int)e;
        return;
      }
      ++done_tasks;
    }
  }
  ~HostTrsm() {
    {
      std::lock_guard<std::mutex> lk(mu);
      quit = true;
    }
    cv_go.notify_all();
    for (auto& th : pool) th.join();
    if (s) cudaStreamDestroy(s);
    if (hX) cudaFreeHost(hX);
    if (hL) cudaFreeHost(hL);
    if (hD) cudaFreeHost(hD);
    if (h_epoch) cudaFreeHost(h_epoch);
  }
};

int host_trsm_create(HostTrsm** out, int device, int nb, int bs, int nthreads, int64_t ntiles, double* tiles,
                     const double* d_dinv, int* d_host_flags, const int* h_ready,
                     const std::vector<std::pair<int, int>>& tasks) {
  auto* h = new HostTrsm();
  h->device = device;
  h->nb = nb;
  h->bs = bs;
  h->nthreads = nthreads > 0 ? nthreads : (int)std::max(1u, std::thread::hardware_concurrency());
  h->ntiles = ntiles;
  h->tiles = tiles;
  h->d_dinv = d_dinv;
  h->d_host_flags = d_host_flags;
  h->ready = h_ready;
  h->tasks = tasks;
  if (h->init()) {
    delete h;
    return -9;
  }
  *out = h;
  return 0;
}

void host_trsm_start(HostTrsm* h, unsigned epoch) {
  h->epoch = epoch;
  h->status = 0;
  h->done_tasks = 0;
  h->stop = false;
  h->driver = std::thread([h] {
    cudaSetDevice(h->device);
    h->run();
  });
}

int host_trsm_finish(HostTrsm* h, bool abort) {
  if (abort) h->stop = true;
  if (h->driver.joinable()) h->driver.join();
  return h->status;
}

int host_trsm_count(const HostTrsm* h) { return (int)h->tasks.size(); }
int host_trsm_done(const HostTrsm* h) { return h->done_tasks; }
int host_trsm_threads(const HostTrsm* h) { return h->nthreads; }

void host_trsm_destroy(HostTrsm* h) {
  if (!h) return;
  host_trsm_finish(h, true);
  delete h;
}

// X <- X L^{-T} on the host (the CPU class's kernel), the inverses of L's diagonal blocks
// computed here by substitution on the identity (as the device's J_INV jobs do)
int host_trsm_solve(double* X, const double* L, int nb, int bs) {
  if (nb <= 0 || bs <= 0 || nb % bs || nb % 4 || bs % 8) return -6;
  const int nbb = nb / bs;
  std::vector<double> dinv((size_t)nbb * bs * bs, 0.0);
  for (int b = 0; b < nbb; ++b) {
    const double* Lb = L + (int64_t)b * bs * nb + b * bs;
    double* D = dinv.data() + (size_t)b * bs * bs;
    for (int c = 0; c < bs; ++c)  // column c of inv(L_bb): L_bb x = e_c
      for (int r = c; r < bs; ++r) {
        double v = r == c ? 1.0 : 0.0;
        for (int m = c; m < r; ++m) v -= Lb[(int64_t)r * nb + m] * D[(size_t)m * bs + c];
        D[(size_t)r * bs + c] = v / Lb[(int64_t)r * nb + r];
      }
  }
  std::vector<double> y(4 * (size_t)bs);
  for (int r = 0; r < nb; r += 4) trsm_rows(X, L, dinv.data(), nb, bs, r, y.data());
  return 0;
}

}  // namespace chol

// C-ABI (host only): the CPU class's tile kernel, for tests and the NEXT-3 measurements
extern "C" int chol_cpu_trsm(double* X, const double* L, int64_t nb, int bs) {
  if (!X || !L) return -4;
  return chol::host_trsm_solve(X, L, (int)nb, bs);
}
