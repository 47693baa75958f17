// Host CPU cores as a second resource class for the TRSMs far from the diagonal (hetero.cpp).
#pragma once
#include <cstdint>
#include <utility>
#include <vector>

namespace chol {
struct HostTrsm;
// tasks: (i, k) in Algorithm 1 order; h_ready: host-mapped per-tile "inputs final" epochs
// (written by the device's OUT nodes); d_host_flags: device per-tile epochs the host raises
// after writing L_ik back (watched by the scheduler's watcher warp)
int host_trsm_create(HostTrsm** out, int device, int nb, int bs, int nthreads, int64_t ntiles, double* tiles,
                     const double* d_dinv, int* d_host_flags, const int* h_ready,
                     const std::vector<std::pair<int, int>>& tasks);
void host_trsm_start(HostTrsm* h, unsigned epoch);     // after the factorization kernel is launched
int host_trsm_finish(HostTrsm* h, bool abort);         // join the driver (abort: stop waiting)
int host_trsm_count(const HostTrsm* h);
int host_trsm_done(const HostTrsm* h);
int host_trsm_threads(const HostTrsm* h);
void host_trsm_destroy(HostTrsm* h);
int host_trsm_solve(double* X, const double* L, int nb, int bs);
}  // namespace chol
