// Cycle-level timing of the in-block routines (solve_block, potf2_block) on one CTA.
// Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -std=c++17 -I../../paper_conf_ipps_agullobehkmt15_b200/csrc block_bench.cu -o block_bench
#include <cstdio>
#include <vector>
#include <cmath>
#include "tile_ops.cuh"
using namespace chol;

template <int BS>
__global__ void __launch_bounds__(kThreads, 1) k_bench(double* X, double* L, double* A, int ld, int* info, long long* cyc, int reps) {
  auto c = make_ctx<BS>(nullptr, nullptr, ld, 1);
  Acc<BS> acc;
  long long t0 = clock64();
  for (int r = 0; r < reps; ++r) solve_block(c, X, ld, L, ld);
  long long t1 = clock64();
  for (int r = 0; r < reps; ++r) potf2_block(c, A, ld, 0, info);
  __syncthreads();
  long long t2 = clock64();
  if (threadIdx.x == 0) { cyc[0] = (t1 - t0) / reps; cyc[1] = (t2 - t1) / reps; }
}

int main() {
  constexpr int BS = 96;
  const int ld = BS;
  std::vector<double> hX(BS * BS), hL(BS * BS, 0.0), hA(BS * BS);
  for (int i = 0; i < BS; ++i)
    for (int j = 0; j < BS; ++j) {
      hX[i * BS + j] = 0.001 * ((i * 7 + j * 3) % 11);
      hL[i * BS + j] = (j < i) ? 0.01 * ((i + j) % 5) : (j == i ? 2.0 : 0.0);
      hA[i * BS + j] = (i == j) ? BS : 0.1 / (1 + abs(i - j));
    }
  double *X, *L, *A; int* info; long long* cyc;
  cudaMalloc(&X, BS * BS * 8); cudaMalloc(&L, BS * BS * 8); cudaMalloc(&A, BS * BS * 8);
  cudaMalloc(&info, 4); cudaMalloc(&cyc, 16);
  cudaMemcpy(X, hX.data(), BS * BS * 8, cudaMemcpyHostToDevice);
  cudaMemcpy(L, hL.data(), BS * BS * 8, cudaMemcpyHostToDevice);
  cudaMemcpy(A, hA.data(), BS * BS * 8, cudaMemcpyHostToDevice);
  const int smem = Cfg<BS>::kSmemBytes;
  cudaFuncSetAttribute(k_bench<BS>, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
  for (int reps : {1, 4}) {
    k_bench<BS><<<1, kThreads, smem>>>(X, L, A, ld, info, cyc, reps);
    cudaError_t e = cudaDeviceSynchronize();
    long long h[2];
    cudaMemcpy(h, cyc, 16, cudaMemcpyDeviceToHost);
    printf("{\"reps\": %d, \"err\": \"%s\", \"solve_block_cycles\": %lld, \"potf2_block_cycles\": %lld}\n", reps, cudaGetErrorString(e), h[0], h[1]);
  }
  return 0;
}
