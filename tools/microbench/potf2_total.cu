// potf2_block alone on one CTA (BS = 96): clock64 from the first to the last barrier,
// best of 20 launches (no phase stamps: they add global round trips to the chain).
// Build against a tile_ops.cuh with -I (A/B of two versions).
#include <cstdio>
#include <vector>
#include "tile_ops.cuh"
using namespace chol;
__device__ long long g_cyc;
__global__ void __launch_bounds__(kThreads, 1) k_bench(double* A, int ld, int* info) {
  auto c = make_ctx<96>(nullptr, nullptr, ld, 1);
  __syncthreads();
  const long long t0 = clock64();
  potf2_block(c, A, ld, 0, info);
  __syncthreads();
  if (threadIdx.x == 0) g_cyc = clock64() - t0;
}
int main() {
  const int BS = 96, ld = BS;
  std::vector<double> hA(BS * BS);
  for (int i = 0; i < BS; ++i)
    for (int j = 0; j < BS; ++j) hA[i * BS + j] = (i == j) ? BS : 0.1 / (1 + abs(i - j));
  double* A; int* info;
  cudaMalloc(&A, BS * BS * 8); cudaMalloc(&info, 4);
  cudaFuncSetAttribute(k_bench, cudaFuncAttributeMaxDynamicSharedMemorySize, Cfg<96>::kSmemBytes);
  long long best = 1ll << 60;
  for (int rep = 0; rep < 20; ++rep) {
    cudaMemcpy(A, hA.data(), BS * BS * 8, cudaMemcpyHostToDevice);
    k_bench<<<1, kThreads, Cfg<96>::kSmemBytes>>>(A, ld, info);
    cudaDeviceSynchronize();
    long long cyc;
    cudaMemcpyFromSymbol(&cyc, g_cyc, 8);
    if (cyc < best) best = cyc;
  }
  std::vector<double> L(BS * BS);
  cudaMemcpy(L.data(), A, BS * BS * 8, cudaMemcpyDeviceToHost);
  double cs = 0;
  for (double v : L) cs += v;
  printf("potf2_block BS=96: best %lld cycles (%s), checksum %.17g\n", best, cudaGetErrorString(cudaGetLastError()), cs);
  return 0;
}
