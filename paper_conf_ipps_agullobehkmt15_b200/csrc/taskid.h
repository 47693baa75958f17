// Dense task numbering shared by the planner (host) and the kernels (device).
// Fig. 1 names: POTRF_k, TRSM_i_k, SYRK_j_k, GEMM_i_j_k.
// Ids: [0, N) POTRF | [N, N+NT) TRSM | [N+NT, N+2NT) SYRK | [N+2NT, ...) GEMM,
// NT = N(N-1)/2; inside a type, ordered by k, then by (j, i) as Algorithm 1
// (L172-181) visits them.
#pragma once
#include <stdint.h>

#ifdef __CUDACC__
#define CHOL_HD __host__ __device__ __forceinline__
#else
#define CHOL_HD inline
#endif

namespace chol {

// tile (i, j), i >= j, of the packed lower tile store
CHOL_HD int64_t tile_index(int64_t i, int64_t j) { return i * (i + 1) / 2 + j; }

enum TaskType : int { T_POTRF = 0, T_TRSM = 1, T_SYRK = 2, T_GEMM = 3 };

CHOL_HD int64_t n_trsm(int64_t N) { return N * (N - 1) / 2; }
CHOL_HD int64_t n_gemm(int64_t N) { return N * (N - 1) * (N - 2) / 6; }
CHOL_HD int64_t n_tasks(int64_t N) { return N + 2 * n_trsm(N) + n_gemm(N); }
CHOL_HD int64_t c3(int64_t m) { return m * (m - 1) * (m - 2) / 6; }

// index of (i, k), i > k, among the pairs ordered by k then i
CHOL_HD int64_t tri_index(int64_t N, int64_t i, int64_t k) { return k * (2 * N - k - 1) / 2 + (i - k - 1); }

CHOL_HD int64_t id_potrf(int64_t /*N*/, int64_t k) { return k; }
CHOL_HD int64_t id_trsm(int64_t N, int64_t i, int64_t k) { return N + tri_index(N, i, k); }
CHOL_HD int64_t id_syrk(int64_t N, int64_t j, int64_t k) { return N + n_trsm(N) + tri_index(N, j, k); }
CHOL_HD int64_t id_gemm(int64_t N, int64_t i, int64_t j, int64_t k) {
  // sum_{k'<k} C(N-1-k', 2) = C(N,3) - C(N-k,3); then (j, i) pairs with k < j < i < N
  const int64_t before_k = c3(N) - c3(N - k);
  const int64_t before_j = (j - k - 1) * (2 * N - 2 - j - k) / 2;
  return N + 2 * n_trsm(N) + before_k + before_j + (i - j - 1);
}

}  // namespace chol
