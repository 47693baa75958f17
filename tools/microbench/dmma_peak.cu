// FP64 peak microbenchmark for B200 (sm_100a): DFMA vs DMMA (mma.sync .f64)
// shapes m8n8k4 / m16n8k4 / m16n8k8 / m16n8k16, plus a fragment-layout check
// for each DMMA shape against a host triple loop.
//
// Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o dmma_peak dmma_peak.cu
// Prints one JSON object per line.
#include <cstdio>
#include <cstdlib>
#include <cmath>
#include <vector>
#include <cuda_runtime.h>

#define CK(x) do { cudaError_t e = (x); if (e != cudaSuccess) { \
  fprintf(stderr, "CUDA %s at %s:%d\n", cudaGetErrorString(e), __FILE__, __LINE__); exit(1);} } while (0)

// ---------------------------------------------------------------- DMMA ops
__device__ __forceinline__ void mma884(double (&d)[2], double a, double b) {
  asm volatile("mma.sync.aligned.m8n8k4.row.col.f64.f64.f64.f64 {%0,%1}, {%2}, {%3}, {%0,%1};\n"
               : "+d"(d[0]), "+d"(d[1]) : "d"(a), "d"(b));
}
__device__ __forceinline__ void mma1684(double (&d)[4], const double (&a)[2], double b) {
  asm volatile("mma.sync.aligned.m16n8k4.row.col.f64.f64.f64.f64 {%0,%1,%2,%3}, {%4,%5}, {%6}, {%0,%1,%2,%3};\n"
               : "+d"(d[0]), "+d"(d[1]), "+d"(d[2]), "+d"(d[3]) : "d"(a[0]), "d"(a[1]), "d"(b));
}
__device__ __forceinline__ void mma1688(double (&d)[4], const double (&a)[4], const double (&b)[2]) {
  asm volatile("mma.sync.aligned.m16n8k8.row.col.f64.f64.f64.f64 {%0,%1,%2,%3}, {%4,%5,%6,%7}, {%8,%9}, {%0,%1,%2,%3};\n"
               : "+d"(d[0]), "+d"(d[1]), "+d"(d[2]), "+d"(d[3])
               : "d"(a[0]), "d"(a[1]), "d"(a[2]), "d"(a[3]), "d"(b[0]), "d"(b[1]));
}
__device__ __forceinline__ void mma16816(double (&d)[4], const double (&a)[8], const double (&b)[4]) {
  asm volatile("mma.sync.aligned.m16n8k16.row.col.f64.f64.f64.f64 {%0,%1,%2,%3}, "
               "{%4,%5,%6,%7,%8,%9,%10,%11}, {%12,%13,%14,%15}, {%0,%1,%2,%3};\n"
               : "+d"(d[0]), "+d"(d[1]), "+d"(d[2]), "+d"(d[3])
               : "d"(a[0]), "d"(a[1]), "d"(a[2]), "d"(a[3]), "d"(a[4]), "d"(a[5]), "d"(a[6]), "d"(a[7]),
                 "d"(b[0]), "d"(b[1]), "d"(b[2]), "d"(b[3]));
}

// ---------------------------------------------------------------- peak kernels
constexpr int ACC = 8;  // independent accumulators per thread/warp

__global__ void k_dfma(double* out, int iters, double x) {
  double acc[ACC];
#pragma unroll
  for (int i = 0; i < ACC; ++i) acc[i] = threadIdx.x * 1e-9 + i;
  double y = x * 0.999;
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < ACC; ++i) acc[i] = fma(acc[i], x, y);
  }
  double s = 0;
#pragma unroll
  for (int i = 0; i < ACC; ++i) s += acc[i];
  if (s == 12345.678) out[0] = s;
}

__global__ void k_m884(double* out, int iters, double x) {
  double d[ACC][2];
#pragma unroll
  for (int i = 0; i < ACC; ++i) d[i][0] = d[i][1] = threadIdx.x * 1e-9 + i;
  double a = x, b = x * 0.5;
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < ACC; ++i) mma884(d[i], a, b);
  }
  double s = 0;
#pragma unroll
  for (int i = 0; i < ACC; ++i) s += d[i][0] + d[i][1];
  if (s == 12345.678) out[0] = s;
}

__global__ void k_m1684(double* out, int iters, double x) {
  double d[ACC][4];
#pragma unroll
  for (int i = 0; i < ACC; ++i) d[i][0] = d[i][1] = d[i][2] = d[i][3] = threadIdx.x * 1e-9 + i;
  double a[2] = {x, x * 0.3}, b = x * 0.5;
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < ACC; ++i) mma1684(d[i], a, b);
  }
  double s = 0;
#pragma unroll
  for (int i = 0; i < ACC; ++i) s += d[i][0] + d[i][1] + d[i][2] + d[i][3];
  if (s == 12345.678) out[0] = s;
}

__global__ void k_m1688(double* out, int iters, double x) {
  double d[ACC][4];
#pragma unroll
  for (int i = 0; i < ACC; ++i) d[i][0] = d[i][1] = d[i][2] = d[i][3] = threadIdx.x * 1e-9 + i;
  double a[4] = {x, x * 0.3, x * 0.7, x * 0.1}, b[2] = {x * 0.5, x * 0.25};
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < ACC; ++i) mma1688(d[i], a, b);
  }
  double s = 0;
#pragma unroll
  for (int i = 0; i < ACC; ++i) s += d[i][0] + d[i][1] + d[i][2] + d[i][3];
  if (s == 12345.678) out[0] = s;
}

__global__ void k_m16816(double* out, int iters, double x) {
  double d[ACC][4];
#pragma unroll
  for (int i = 0; i < ACC; ++i) d[i][0] = d[i][1] = d[i][2] = d[i][3] = threadIdx.x * 1e-9 + i;
  double a[8], b[4];
#pragma unroll
  for (int i = 0; i < 8; ++i) a[i] = x * (i + 1) * 0.1;
#pragma unroll
  for (int i = 0; i < 4; ++i) b[i] = x * (i + 1) * 0.2;
  for (int it = 0; it < iters; ++it) {
#pragma unroll
    for (int i = 0; i < ACC; ++i) mma16816(d[i], a, b);
  }
  double s = 0;
#pragma unroll
  for (int i = 0; i < ACC; ++i) s += d[i][0] + d[i][1] + d[i][2] + d[i][3];
  if (s == 12345.678) out[0] = s;
}

// ---------------------------------------------------------------- layout check
// A is MxK row-major, B is KxN stored as B[k][n] (row-major KxN), D = A*B (MxN row-major).
// g = lane>>2, t = lane&3.  Assumed fragment maps (PTX ISA, f64 mma):
//  m8n8k4 : a0=(g,t)            b0=(k=t,n=g)                 c_i=(g, 2t+i)
//  m16n8k4: a_i=(g+8i, t)       b0=(t,g)                     c_i=(g+8*(i>>1), 2t+(i&1))
//  m16n8k8: a_i=(g+8*(i&1), t+4*(i>>1))  b_i=(t+4i, g)        c as m16n8k4
//  m16n8k16: a_i=(g+8*(i&1), t+4*(i>>1)) b_i=(t+4i, g)        c as m16n8k4
template <int M, int N, int K>
__global__ void k_layout(const double* A, const double* B, double* D) {
  int lane = threadIdx.x, g = lane >> 2, t = lane & 3;
  if (M == 8) {
    double d[2] = {0, 0};
    mma884(d, A[g * K + t], B[t * N + g]);
    D[g * N + 2 * t] = d[0];
    D[g * N + 2 * t + 1] = d[1];
    return;
  }
  double d[4] = {0, 0, 0, 0};
  if (K == 4) {
    double a[2] = {A[g * K + t], A[(g + 8) * K + t]};
    mma1684(d, a, B[t * N + g]);
  } else if (K == 8) {
    double a[4], b[2];
    for (int i = 0; i < 4; ++i) a[i] = A[(g + 8 * (i & 1)) * K + t + 4 * (i >> 1)];
    for (int i = 0; i < 2; ++i) b[i] = B[(t + 4 * i) * N + g];
    mma1688(d, a, b);
  } else {
    double a[8], b[4];
    for (int i = 0; i < 8; ++i) a[i] = A[(g + 8 * (i & 1)) * K + t + 4 * (i >> 1)];
    for (int i = 0; i < 4; ++i) b[i] = B[(t + 4 * i) * N + g];
    mma16816(d, a, b);
  }
  for (int i = 0; i < 4; ++i) D[(g + 8 * (i >> 1)) * N + 2 * t + (i & 1)] = d[i];
}

template <int M, int N, int K>
void check_layout(const char* name) {
  std::vector<double> A(M * K), B(K * N), D(M * N), R(M * N, 0.0);
  for (int i = 0; i < M * K; ++i) A[i] = (double)((i * 7 + 3) % 17) - 8.0;
  for (int i = 0; i < K * N; ++i) B[i] = (double)((i * 5 + 1) % 13) - 6.0;
  for (int m = 0; m < M; ++m)
    for (int n = 0; n < N; ++n)
      for (int k = 0; k < K; ++k) R[m * N + n] += A[m * K + k] * B[k * N + n];
  double *dA, *dB, *dD;
  CK(cudaMalloc(&dA, A.size() * 8)); CK(cudaMalloc(&dB, B.size() * 8)); CK(cudaMalloc(&dD, D.size() * 8));
  CK(cudaMemcpy(dA, A.data(), A.size() * 8, cudaMemcpyHostToDevice));
  CK(cudaMemcpy(dB, B.data(), B.size() * 8, cudaMemcpyHostToDevice));
  k_layout<M, N, K><<<1, 32>>>(dA, dB, dD);
  CK(cudaGetLastError());
  CK(cudaMemcpy(D.data(), dD, D.size() * 8, cudaMemcpyDeviceToHost));
  int bad = 0;
  for (int i = 0; i < M * N; ++i) bad += (D[i] != R[i]);
  printf("{\"layout\": \"%s\", \"mismatches\": %d}\n", name, bad);
  cudaFree(dA); cudaFree(dB); cudaFree(dD);
}

template <typename F>
void time_peak(const char* name, F kern, double flop_per_thread_iter, int blocks_per_sm, int threads) {
  int sms = 0;
  CK(cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0));
  double* out; CK(cudaMalloc(&out, 8));
  int iters = 20000;
  int grid = sms * blocks_per_sm;
  kern<<<grid, threads>>>(out, 100, 1.0000001);
  CK(cudaDeviceSynchronize());
  cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
  float best = 1e30f;
  for (int rep = 0; rep < 5; ++rep) {
    cudaEventRecord(e0);
    kern<<<grid, threads>>>(out, iters, 1.0000001);
    cudaEventRecord(e1);
    CK(cudaEventSynchronize(e1));
    float ms; cudaEventElapsedTime(&ms, e0, e1);
    if (ms < best) best = ms;
  }
  double flops = flop_per_thread_iter * (double)iters * grid * threads;
  printf("{\"kernel\": \"%s\", \"blocks_per_sm\": %d, \"threads\": %d, \"ms\": %.3f, \"tflops\": %.3f}\n",
         name, blocks_per_sm, threads, best, flops / best / 1e9);
  cudaFree(out);
}

int main() {
  check_layout<8, 8, 4>("m8n8k4");
  check_layout<16, 8, 4>("m16n8k4");
  check_layout<16, 8, 8>("m16n8k8");
  check_layout<16, 8, 16>("m16n8k16");
  // flop per thread per iteration: DFMA: ACC*2; mma MxNxK per warp: 2*M*N*K*ACC/32 per thread
  for (int bps : {1, 2, 4}) {
    time_peak("dfma", k_dfma, ACC * 2.0, bps, 256);
    time_peak("m8n8k4", k_m884, ACC * 2.0 * 8 * 8 * 4 / 32, bps, 256);
    time_peak("m16n8k4", k_m1684, ACC * 2.0 * 16 * 8 * 4 / 32, bps, 256);
    time_peak("m16n8k8", k_m1688, ACC * 2.0 * 16 * 8 * 8 / 32, bps, 256);
    time_peak("m16n8k16", k_m16816, ACC * 2.0 * 16 * 8 * 16 / 32, bps, 256);
  }
  return 0;
}
