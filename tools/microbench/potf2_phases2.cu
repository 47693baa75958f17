// Per-phase timing of potf2_block (one CTA, BS = 96) with low-overhead stamps: lane 0 of
// each warp writes the low 32 bits of clock64 into a shared-memory table (no global round
// trips on the chain).  Stamps: 0 pivot published (row warps), 1 panel stored, 2 panel
// barrier passed, 3 next diagonal block handed over (owner), 4 updates done, 5 factor warp
// got its block, 6 factor done.  Printed per panel relative to the start.
#include <cstdio>
#include <vector>
__shared__ unsigned s_st[8][7][12];
__shared__ int s_cnt[8][7];
#define POTF2_STAMP(id)                                                 \
  do {                                                                  \
    if ((threadIdx.x & 31) == 0) {                                      \
      const unsigned t_ = (unsigned)clock64();                          \
      const int w_ = threadIdx.x >> 5, k_ = s_cnt[w_][id]++;            \
      if (k_ < 12) s_st[w_][id][k_] = t_;                               \
    }                                                                   \
  } while (0)
#include "tile_ops.cuh"
using namespace chol;
__device__ unsigned g_st[8][7][12];
__device__ unsigned g_t0, g_t1;
__global__ void __launch_bounds__(kThreads, 1) k_bench(double* A, int ld, int* info) {
  if (threadIdx.x < 56) s_cnt[threadIdx.x / 7][threadIdx.x % 7] = 0;
  auto c = make_ctx<96>(nullptr, nullptr, ld, 1);
  __syncthreads();
  const unsigned t0 = (unsigned)clock64();
  potf2_block(c, A, ld, 0, info);
  __syncthreads();
  const unsigned t1 = (unsigned)clock64();
  for (int e = threadIdx.x; e < 8 * 7 * 12; e += blockDim.x) (&g_st[0][0][0])[e] = (&s_st[0][0][0])[e] - t0;
  if (threadIdx.x == 0) { g_t0 = t0; g_t1 = t1 - t0; }
}
int main() {
  const int BS = 96, ld = BS;
  std::vector<double> hA(BS * BS);
  for (int i = 0; i < BS; ++i)
    for (int j = 0; j < BS; ++j) hA[i * BS + j] = (i == j) ? BS : 0.1 / (1 + abs(i - j));
  double* A; int* info;
  cudaMalloc(&A, BS * BS * 8); cudaMalloc(&info, 4);
  const int smem = Cfg<96>::kSmemBytes;
  cudaFuncSetAttribute(k_bench, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
  unsigned best = ~0u, st[8][7][12], tot = 0;
  for (int rep = 0; rep < 10; ++rep) {
    cudaMemcpy(A, hA.data(), BS * BS * 8, cudaMemcpyHostToDevice);
    k_bench<<<1, kThreads, smem>>>(A, ld, info);
    cudaDeviceSynchronize();
    cudaMemcpyFromSymbol(&tot, g_t1, 4);
    if (tot < best) { best = tot; cudaMemcpyFromSymbol(st, g_st, sizeof(st)); }
  }
  printf("err %s total %u cycles\n", cudaGetErrorString(cudaGetLastError()), best);
  for (int p = 0; p < 12; ++p) {
    const int nr = p + 1 < 6 ? p + 1 : 10 - p, nw = nr < 3 ? nr : nr + 1;  // owner warp of row block p+1
    printf("panel %2d  w7 got %6u done %6u | w0 piv %6u stored %6u pbar %6u upd %6u | owner w%d piv %6u handoff %6u\n", p,
           st[7][5][p], st[7][6][p], st[0][0][p], st[0][1][p], st[0][2][p], p < 11 ? st[0][4][p] : 0, nw,
           p < 11 ? st[nw & 7][0][p] : 0, p < 11 ? st[nw & 7][3][(p + 1 < 6 || nr == 0) ? 0 : 1] : 0);
  }
  return 0;
}
