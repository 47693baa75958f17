// Per-phase timing of potf2_block (one CTA, BS = 96): clock64 stamps through the
// POTF2_STAMP hook.  Per panel, for warp w (lane 0) and the factor warp 7:
//   0 after barrier "L_pp published", 1 rows solved, 2 after barrier "panel published",
//   3 next diagonal block handed over (owner warp), 4 updates done, 5 factor warp got the
//   block, 6 factor warp done.  Printed as cycles relative to the kernel start.
#include <cstdio>
#include <vector>
__device__ long long g_st[8][8][16];  // [warp][stamp][panel-ish counter]
__device__ int g_cnt[8][8];
#define POTF2_STAMP(id)                                                         \
  do {                                                                          \
    if ((threadIdx.x & 31) == 0) {                                              \
      const int w_ = threadIdx.x >> 5, k_ = g_cnt[w_][id]++;                     \
      if (k_ < 16) g_st[w_][id][k_] = clock64();                                \
    }                                                                           \
  } while (0)
#include "tile_ops.cuh"
using namespace chol;
__device__ long long g_t0;
__global__ void __launch_bounds__(kThreads, 1) k_bench(double* A, int ld, int* info) {
  auto c = make_ctx<96>(nullptr, nullptr, ld, 1);
  if (threadIdx.x == 0) g_t0 = clock64();
  potf2_block(c, A, ld, 0, info);
}
int main() {
  const int BS = 96, ld = BS;
  std::vector<double> hA(BS * BS);
  for (int i = 0; i < BS; ++i)
    for (int j = 0; j < BS; ++j) hA[i * BS + j] = (i == j) ? BS : 0.1 / (1 + abs(i - j));
  double* A; int* info;
  cudaMalloc(&A, BS * BS * 8); cudaMalloc(&info, 4);
  cudaFuncSetAttribute(k_bench, cudaFuncAttributeMaxDynamicSharedMemorySize, Cfg<96>::kSmemBytes);
  for (int rep = 0; rep < 2; ++rep) {
    cudaMemcpy(A, hA.data(), BS * BS * 8, cudaMemcpyHostToDevice);
    cudaMemset(info, 0x7f, 4);
    int z[64] = {0};
    cudaMemcpyToSymbol(g_cnt, z, sizeof(z));
    k_bench<<<1, kThreads, Cfg<96>::kSmemBytes>>>(A, ld, info);
    cudaDeviceSynchronize();
  }
  long long st[8][8][16], t0;
  cudaMemcpyFromSymbol(st, g_st, sizeof(st));
  cudaMemcpyFromSymbol(&t0, g_t0, 8);
  printf("err %s\n", cudaGetErrorString(cudaGetLastError()));
  for (int p = 0; p < 12; ++p) {
    printf("panel %2d  w0: bar %6lld solved %6lld bar2 %6lld upd %6lld | w%d handoff %6lld | w7 got %6lld done %6lld\n", p,
           st[0][0][p] - t0, st[0][1][p] - t0, st[0][2][p] - t0, st[0][4][p] - t0, p + 1 < 6 ? p + 1 : 10 - p,
           st[(p + 1 < 6 ? p + 1 : 10 - p) & 7][3][0] - t0, st[7][5][p] - t0, st[7][6][p] - t0);
  }
  return 0;
}
