// Day-1 microbenchmarks on B200: latencies that set the
// sweep kernel's latency roof and the HBM write roof.  Not part of the product.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

#define CK(x) do { cudaError_t e = (x); if (e != cudaSuccess) { printf("CUDA %s at %d\n", cudaGetErrorString(e), __LINE__); return 1; } } while (0)

__global__ void chain_viaddmax(int* out, int n, int g, long long* cyc) {
  int a = threadIdx.x, b = 3;
  long long t0 = clock64();
  for (int i = 0; i < n; ++i) {
#pragma unroll
    for (int u = 0; u < 16; ++u) a = __viaddmax_s32(a, g, b + u);
  }
  long long t1 = clock64();
  out[threadIdx.x] = a; if (threadIdx.x == 0) *cyc = t1 - t0;
}
__global__ void chain_vimax3(int* out, int n, long long* cyc) {
  int a = threadIdx.x, b = 3, c = 5;
  long long t0 = clock64();
  for (int i = 0; i < n; ++i) {
#pragma unroll
    for (int u = 0; u < 16; ++u) { a = __vimax3_s32(a, b + u, c - u); }
  }
  long long t1 = clock64();
  out[threadIdx.x] = a; if (threadIdx.x == 0) *cyc = t1 - t0;
}
__global__ void chain_ffma(float* out, int n, float A, float c, long long* cyc) {
  float x = threadIdx.x * 1e-3f;
  long long t0 = clock64();
  for (int i = 0; i < n; ++i) {
#pragma unroll
    for (int u = 0; u < 16; ++u) x = __fmaf_rn(x, A, c);
  }
  long long t1 = clock64();
  out[threadIdx.x] = x; if (threadIdx.x == 0) *cyc = t1 - t0;
}
__global__ void chain_shfl(int* out, int n, long long* cyc) {
  int a = threadIdx.x;
  long long t0 = clock64();
  for (int i = 0; i < n; ++i) {
#pragma unroll
    for (int u = 0; u < 16; ++u) a = __shfl_up_sync(0xffffffffu, a, 1) + 1;
  }
  long long t1 = clock64();
  out[threadIdx.x] = a; if (threadIdx.x == 0) *cyc = t1 - t0;
}
// shfl + viaddmax chain (one lane-to-lane hop of the sweep)
__global__ void chain_shfl_max(int* out, int n, long long* cyc) {
  int a = threadIdx.x;
  long long t0 = clock64();
  for (int i = 0; i < n; ++i) {
#pragma unroll
    for (int u = 0; u < 16; ++u) a = __viaddmax_s32(__shfl_up_sync(0xffffffffu, a, 1), -1, u);
  }
  long long t1 = clock64();
  out[threadIdx.x] = a; if (threadIdx.x == 0) *cyc = t1 - t0;
}

// LL (value,tag) ping-pong between CTA 0 and CTA 1 through global memory.
__global__ void ll_pingpong(unsigned long long* slot, int iters, long long* cyc) {
  volatile unsigned long long* s = slot;
  if (threadIdx.x != 0) return;
  long long t0 = clock64();
  for (int i = 0; i < iters; ++i) {
    if (blockIdx.x == 0) {
      s[0] = ((unsigned long long)(2 * i + 1) << 32) | 7u;
      while ((s[16] >> 32) != (unsigned long long)(2 * i + 2)) {}
    } else {
      while ((s[0] >> 32) != (unsigned long long)(2 * i + 1)) {}
      s[16] = ((unsigned long long)(2 * i + 2) << 32) | 9u;
    }
  }
  long long t1 = clock64();
  if (blockIdx.x == 0) *cyc = t1 - t0;
}
// release/acquire flag ping-pong (gpu scope)
__global__ void relacq_pingpong(int* flag, int iters, long long* cyc) {
  if (threadIdx.x != 0) return;
  long long t0 = clock64();
  for (int i = 0; i < iters; ++i) {
    int v;
    if (blockIdx.x == 0) {
      asm volatile("st.release.gpu.global.b32 [%0], %1;" :: "l"(flag), "r"(2 * i + 1) : "memory");
      do { asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(flag + 32) : "memory"); } while (v != 2 * i + 2);
    } else {
      do { asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(flag) : "memory"); } while (v != 2 * i + 1);
      asm volatile("st.release.gpu.global.b32 [%0], %1;" :: "l"(flag + 32), "r"(2 * i + 2) : "memory");
    }
  }
  long long t1 = clock64();
  if (blockIdx.x == 0) *cyc = t1 - t0;
}
// smem ping-pong between warp 0 and warp 1 (volatile 64-bit LL in shared)
__global__ void smem_pingpong(int iters, long long* cyc) {
  __shared__ unsigned long long s[64];
  if (threadIdx.x == 0) { s[0] = 0; s[32] = 0; }
  __syncthreads();
  volatile unsigned long long* v = s;
  int w = threadIdx.x / 32, l = threadIdx.x % 32;
  if (l != 0) return;
  long long t0 = clock64();
  for (int i = 0; i < iters; ++i) {
    if (w == 0) {
      v[0] = ((unsigned long long)(2 * i + 1) << 32);
      while ((v[32] >> 32) != (unsigned long long)(2 * i + 2)) {}
    } else {
      while ((v[0] >> 32) != (unsigned long long)(2 * i + 1)) {}
      v[32] = ((unsigned long long)(2 * i + 2) << 32);
    }
  }
  long long t1 = clock64();
  if (w == 0) *cyc = t1 - t0;
}
// write-only bandwidth, st.global.v4
__global__ void write_v4(int4* p, size_t n16) {
  size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x, st = (size_t)gridDim.x * blockDim.x;
  for (; i < n16; i += st) p[i] = make_int4((int)i, 1, 2, 3);
}

int main() {
  cudaDeviceProp pr; CK(cudaGetDeviceProperties(&pr, 0));
  int clk = 0; cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, 0);
  printf("{\"name\":\"%s\",\"sms\":%d,\"smem_optin\":%zu,\"regs_per_sm\":%d,\"l2\":%d,\"clock_khz\":%d}\n", pr.name,
         pr.multiProcessorCount, pr.sharedMemPerBlockOptin, pr.regsPerMultiprocessor, pr.l2CacheSize, clk);
  int* d_i; float* d_f; long long* d_c; long long h;
  CK(cudaMalloc(&d_i, 4096)); CK(cudaMalloc(&d_f, 4096)); CK(cudaMalloc(&d_c, 64));
  const int n = 4096; const double ops = 16.0 * n;
  chain_viaddmax<<<1, 32>>>(d_i, n, -1, d_c); CK(cudaDeviceSynchronize());
  chain_viaddmax<<<1, 32>>>(d_i, n, -1, d_c); CK(cudaMemcpy(&h, d_c, 8, cudaMemcpyDeviceToHost));
  printf("lat_viaddmax_cyc %.2f\n", h / ops);
  chain_vimax3<<<1, 32>>>(d_i, n, d_c); CK(cudaDeviceSynchronize());
  chain_vimax3<<<1, 32>>>(d_i, n, d_c); CK(cudaMemcpy(&h, d_c, 8, cudaMemcpyDeviceToHost));
  printf("lat_vimax3_cyc %.2f\n", h / ops);
  chain_ffma<<<1, 32>>>(d_f, n, 0.999f, 1e-4f, d_c); CK(cudaDeviceSynchronize());
  chain_ffma<<<1, 32>>>(d_f, n, 0.999f, 1e-4f, d_c); CK(cudaMemcpy(&h, d_c, 8, cudaMemcpyDeviceToHost));
  printf("lat_ffma_cyc %.2f\n", h / ops);
  chain_shfl<<<1, 32>>>(d_i, n, d_c); CK(cudaDeviceSynchronize());
  chain_shfl<<<1, 32>>>(d_i, n, d_c); CK(cudaMemcpy(&h, d_c, 8, cudaMemcpyDeviceToHost));
  printf("lat_shfl_plus_iadd_cyc %.2f\n", h / ops);
  chain_shfl_max<<<1, 32>>>(d_i, n, d_c); CK(cudaDeviceSynchronize());
  chain_shfl_max<<<1, 32>>>(d_i, n, d_c); CK(cudaMemcpy(&h, d_c, 8, cudaMemcpyDeviceToHost));
  printf("lat_shfl_plus_viaddmax_cyc %.2f\n", h / ops);

  unsigned long long* slot; CK(cudaMalloc(&slot, 4096));
  for (int far = 0; far < 2; ++far) {
    CK(cudaMemset(slot, 0, 4096));
    int iters = 2000;
    // 2 CTAs; with grid 2 they typically land on different SMs
    ll_pingpong<<<2, 32>>>(slot, iters, d_c); CK(cudaDeviceSynchronize());
    CK(cudaMemcpy(&h, d_c, 8, cudaMemcpyDeviceToHost));
    printf("ll_global_oneway_cyc %.1f\n", h / (2.0 * iters));
  }
  CK(cudaMemset(slot, 0, 4096));
  relacq_pingpong<<<2, 32>>>((int*)slot, 2000, d_c); CK(cudaDeviceSynchronize());
  CK(cudaMemcpy(&h, d_c, 8, cudaMemcpyDeviceToHost));
  printf("relacq_global_oneway_cyc %.1f\n", h / 4000.0);
  smem_pingpong<<<1, 64>>>(2000, d_c); CK(cudaDeviceSynchronize());
  CK(cudaMemcpy(&h, d_c, 8, cudaMemcpyDeviceToHost));
  printf("smem_ll_oneway_cyc %.1f\n", h / 4000.0);

  size_t bytes = 4ull << 30; int4* big; CK(cudaMalloc(&big, bytes));
  cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
  for (int rep = 0; rep < 3; ++rep) {
    write_v4<<<148 * 8, 256>>>(big, bytes / 16);
  }
  float best = 1e9;
  for (int rep = 0; rep < 10; ++rep) {
    cudaEventRecord(e0); write_v4<<<148 * 8, 256>>>(big, bytes / 16); cudaEventRecord(e1);
    CK(cudaEventSynchronize(e1)); float ms; cudaEventElapsedTime(&ms, e0, e1); if (ms < best) best = ms;
  }
  printf("write_only_4GiB_ms %.4f GBps %.1f\n", best, bytes / (best * 1e-3) / 1e9);
  return 0;
}
