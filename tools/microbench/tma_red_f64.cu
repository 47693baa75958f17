// Does the TMA reduce-add store (cp.reduce.async.bulk.tensor .add, UTMAREDG) support FP64?
// Adds a shared-memory 96 x 16 block of -v to a global FP64 block holding c and checks
// c + (-v) bit for bit.  Build: nvcc -gencode arch=compute_100a,code=sm_100a tma_red_f64.cu -lcuda
#include <cuda.h>
#include <cstdio>
#include <cstdint>
#include <cstring>
#include <vector>
typedef CUresult (*PFN)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*, const cuuint64_t*,
                        const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave, CUtensorMapSwizzle,
                        CUtensorMapL2promotion, CUtensorMapFloatOOBfill);
__global__ void k(const __grid_constant__ CUtensorMap map, const double* v) {
  __shared__ __align__(1024) double buf[96 * 16];
  for (int i = threadIdx.x; i < 96 * 16; i += blockDim.x) {
    const int r = i / 16, c = i % 16;
    // 128B swizzle: 16-byte chunk index ^= row & 7
    const int chunk = (c / 2) ^ (r & 7);
    buf[r * 16 + chunk * 2 + (c & 1)] = -v[i];
  }
  asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
  __syncthreads();
  if (threadIdx.x == 0) {
    uint32_t s = (uint32_t)__cvta_generic_to_shared(buf);
    asm volatile("cp.reduce.async.bulk.tensor.3d.global.shared::cta.add.tile.bulk_group [%0, {%2, %3, %4}], [%1];"
                 ::"l"(&map), "r"(s), "r"(16), "r"(96), "r"(1) : "memory");
    asm volatile("cp.async.bulk.commit_group;" ::: "memory");
    asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
  }
}
int main() {
  const int nb = 192;
  std::vector<double> c(2 * nb * nb), v(96 * 16);
  for (size_t i = 0; i < c.size(); ++i) c[i] = 1.0 + 1e-3 * (double)((i * 2654435761u) % 100000);
  for (size_t i = 0; i < v.size(); ++i) v[i] = 0.37 * (double)((i * 40503u) % 977) / 977.0;
  double *dc, *dv;
  cudaMalloc(&dc, c.size() * 8);
  cudaMalloc(&dv, v.size() * 8);
  cudaMemcpy(dc, c.data(), c.size() * 8, cudaMemcpyHostToDevice);
  cudaMemcpy(dv, v.data(), v.size() * 8, cudaMemcpyHostToDevice);
  void* fn;
  cudaDriverEntryPointQueryResult q;
  cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fn, cudaEnableDefault, &q);
  CUtensorMap map;
  const cuuint64_t dims[3] = {(cuuint64_t)nb, (cuuint64_t)nb, 2};
  const cuuint64_t str[2] = {(cuuint64_t)nb * 8, (cuuint64_t)nb * nb * 8};
  const cuuint32_t box[3] = {16, 96, 1}, es[3] = {1, 1, 1};
  CUresult r = ((PFN)fn)(&map, CU_TENSOR_MAP_DATA_TYPE_FLOAT64, 3, dc, dims, str, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE,
                         CU_TENSOR_MAP_SWIZZLE_128B, CU_TENSOR_MAP_L2_PROMOTION_L2_256B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  k<<<1, 256>>>(map, dv);
  cudaError_t e = cudaDeviceSynchronize();
  std::vector<double> out(c.size());
  cudaMemcpy(out.data(), dc, c.size() * 8, cudaMemcpyDeviceToHost);
  long bad = 0, touched = 0;
  for (int p = 0; p < 2; ++p)
    for (int i = 0; i < nb; ++i)
      for (int j = 0; j < nb; ++j) {
        const size_t x = (size_t)p * nb * nb + (size_t)i * nb + j;
        double want = c[x];
        if (p == 1 && i >= 96 && i < 192 && j >= 16 && j < 32) {
          want = c[x] + (-v[(i - 96) * 16 + (j - 16)]);
          ++touched;
        }
        if (memcmp(&want, &out[x], 8)) ++bad;
      }
  printf("{\"encode\": %d, \"err\": \"%s\", \"touched\": %ld, \"mismatches\": %ld}\n", (int)r, cudaGetErrorString(e),
         touched, bad);
  return 0;
}
