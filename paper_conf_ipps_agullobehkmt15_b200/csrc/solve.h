// Triangular solves with the tile-store factor (solve.cu).
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include <algorithm>

namespace chol {
struct SolveArgs {
  const double* tiles;  // packed lower tile store holding L (row-major nb x nb tiles)
  int64_t n;
  int nb, sb;           // tile size, block size (96 / 64 / 32)
  double* inv;          // 3 (n / sb) sb x sb blocks: inverses of the diagonal blocks of L, then
                        // the forward and backward chain matrices (solve.cu, k_diag_aux)
  bool inv_valid;       // inverses already computed for this factor
  double* W;            // right-hand sides, n x ldw row-major, overwritten by the solution
  int ldw, nchunks;     // ldw = rc * nchunks
  int rc;               // right-hand-side columns per work item: 1 (nrhs = 1), 8 (nrhs <= 8) or 32
  int* ctl;             // 2 + 2 * (n / sb) * nchunks ints of control (counters, flags)
  int sms;
  double* chain;        // nrhs = 1: 2 n doubles (forward / backward block results, polled), or null
  uint64_t* trace;      // development: 2 * (n / sb) * nchunks items x 6 u64 (solve.cu), or null
};
cudaError_t solve_run(const SolveArgs& a, cudaStream_t s, int* nlaunch);
}  // namespace chol
