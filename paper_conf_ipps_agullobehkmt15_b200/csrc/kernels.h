// Launchers shared by the C-ABI (api.cu) and the kernels (kernels.cu, scheduler.cu).
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>
#include <stdint.h>

namespace chol {

struct StepParams {
  double* tiles;
  int nb, N;
  int k, b;      // step k; POTRF inner step b
  int i0, j0;    // first TRSM row tile / single-task indices
  int mode;      // k_update mode (0 all, 1 single, 2 GEMM only, 3 SYRK only)
  int* info;     // device int, atomicMin of the failing column (INT_MAX = none)
  uint64_t* tr_t0;          // per-task min start (ns since *tr_base), or null
  uint64_t* tr_t1;          // per-task max (end << 16 | smid)
  const uint64_t* tr_base;  // globaltimer at factorization start
  double* dinv;             // [N][nb/BS] BS x BS inverses of the diagonal blocks of L_kk (inverse-form TRSM)
};

cudaError_t prepare_kernels(int bs);
int smem_bytes(int bs);
// count = number of consecutive diagonal tiles (POTRF) / row tiles (TRSM) from p.k / p.i0
cudaError_t launch_potrf(int bs, const CUtensorMap& map, const StepParams& p, int count, cudaStream_t s, int* nl);
// TRSM_{i,k} for i = p.i0 .. p.i0+count-1 (inverse form): k_inv (the inverses of the diagonal
// blocks of L_kk into p.dinv) then one row-slab CTA per (task, slab); dmap maps p.dinv
cudaError_t launch_trsm(int bs, const CUtensorMap& map, const CUtensorMap& dmap, const StepParams& p, int count,
                        cudaStream_t s, int* nl);
cudaError_t launch_update(int bs, const CUtensorMap& map, const StepParams& p, int ntask, cudaStream_t s, int* nl);
cudaError_t launch_stamp(uint64_t* base, cudaStream_t s);
cudaError_t launch_init_info(int* info, cudaStream_t s);
cudaError_t launch_fill_flags(int* flags, int64_t n, int value, cudaStream_t s);
cudaError_t launch_zero_upper_diag(double* tiles, int nb, int N, cudaStream_t s, const int* slots = nullptr,
                                   int count = -1);
cudaError_t launch_generate(double* tiles, int64_t n, int nb, int N, uint64_t seed, int family, cudaStream_t s,
                            const int* slot_tile = nullptr, int64_t nslots = 0);

}  // namespace chol
