// Dependent-chain latencies on sm_100a (cycles per op): DFMA, DMUL, rsqrt(double),
// shfl, DMMA m8n8k4 (accumulator chain), bar.sync (256 threads), LDS.64.
#include <cstdio>
__global__ void k(double* out, long long* cyc, double a, double b, int n) {
  __shared__ double sm[256];
  double x = a + threadIdx.x, y = b;
  sm[threadIdx.x] = x;
  __syncthreads();
  long long t0 = clock64();
  for (int i = 0; i < n; ++i) x = fma(x, y, 1e-9);
  long long t1 = clock64();
  for (int i = 0; i < n; ++i) x = x * y;
  long long t2 = clock64();
  for (int i = 0; i < n; ++i) x = rsqrt(x) + 1.0;
  long long t3 = clock64();
  for (int i = 0; i < n; ++i) x = __shfl_sync(0xffffffffu, x, (threadIdx.x + 1) & 31) + 1.0;
  long long t4 = clock64();
  double c0 = x, c1 = y;
  for (int i = 0; i < n; ++i)
    asm volatile("mma.sync.aligned.m8n8k4.row.col.f64.f64.f64.f64 {%0,%1}, {%2}, {%3}, {%0,%1};" : "+d"(c0), "+d"(c1) : "d"(a), "d"(b));
  long long t5 = clock64();
  for (int i = 0; i < n; ++i) __syncthreads();
  long long t6 = clock64();
  int idx = threadIdx.x;
  double s = 0;
  for (int i = 0; i < n; ++i) { double v = sm[idx]; idx = ((int)v) & 255; s += v; }
  long long t7 = clock64();
  for (int i = 0; i < n; ++i) x = 1.0 / x + 1.0;
  long long t8 = clock64();
  for (int i = 0; i < n; ++i) x = sqrt(x) + 1.0;
  long long t9 = clock64();
  out[threadIdx.x] = x + c0 + c1 + s;
  if (threadIdx.x == 0) {
    cyc[0] = (t1 - t0) / n; cyc[1] = (t2 - t1) / n; cyc[2] = (t3 - t2) / n; cyc[3] = (t4 - t3) / n;
    cyc[4] = (t5 - t4) / n; cyc[5] = (t6 - t5) / n; cyc[6] = (t7 - t6) / n; cyc[7] = (t8 - t7) / n; cyc[8] = (t9 - t8) / n;
  }
}
int main() {
  double* o; long long* c; cudaMalloc(&o, 256 * 8); cudaMalloc(&c, 9 * 8);
  for (int r = 0; r < 2; ++r) k<<<1, 256>>>(o, c, 1.0000001, 0.9999999, 1000);
  long long h[9]; cudaMemcpy(h, c, 72, cudaMemcpyDeviceToHost);
  printf("{\"dfma\": %lld, \"dmul\": %lld, \"rsqrt_f64\": %lld, \"shfl+dadd\": %lld, \"dmma_chain\": %lld, \"bar_sync_256\": %lld, \"lds_chain\": %lld, \"rcp_f64+dadd\": %lld, \"sqrt_f64+dadd\": %lld}\n",
         h[0], h[1], h[2], h[3], h[4], h[5], h[6], h[7], h[8]);
}
