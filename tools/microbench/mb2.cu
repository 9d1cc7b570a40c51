// Per-iteration cost of one 8-byte store flavour inside a dependent ALU loop (1 warp,
// lane 31 stores), to find what throttles the sweep's LL edge publication.
#include <cstdio>
#include <cuda_runtime.h>

template <int MODE>
__global__ void loop(unsigned long long* buf, int n, long long* cyc, int* sink) {
  int a = threadIdx.x;
  long long t0 = clock64();
  for (int i = 0; i < n; ++i) {
    a = __viaddmax_s32(a, 3, i);
    a = __shfl_up_sync(0xffffffffu, a, 1) + 1;
    unsigned long long v = ((unsigned long long)i << 32) | (unsigned)a;
    unsigned long long* p = buf + i;
    if (threadIdx.x == 31) {
      if (MODE == 0) asm volatile("st.relaxed.sys.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
      if (MODE == 1) asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
      if (MODE == 2) asm volatile("st.volatile.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
      if (MODE == 3) asm volatile("st.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
      if (MODE == 4) asm volatile("st.global.cs.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
    }
    if (MODE == 5) {  // every lane stores 16 B coalesced (the row write-out)
      int4* q = reinterpret_cast<int4*>(buf) + (size_t)i * 32 + threadIdx.x;
      *q = make_int4(a, a, a, a);
    }
    if (MODE == 6) {  // ld.relaxed.sys poll (one load per iteration, result consumed)
      unsigned long long w;
      asm volatile("ld.relaxed.sys.global.u64 %0, [%1];" : "=l"(w) : "l"(p) : "memory");
      a += (int)w;
    }
    if (MODE == 7) {  // ld.global.nc byte, consumed next iteration
      a += __ldg(reinterpret_cast<const unsigned char*>(buf) + (i & 4095) + threadIdx.x);
    }
  }
  long long t1 = clock64();
  if (threadIdx.x == 0) { *cyc = t1 - t0; *sink = a; }
}

int main() {
  unsigned long long* buf; long long* cyc; int* sink;
  cudaMalloc(&buf, 64 << 20); cudaMalloc(&cyc, 8); cudaMalloc(&sink, 4);
  cudaMemset(buf, 0, 64 << 20);
  const int n = 20000;
  const char* names[] = {"st.relaxed.sys", "st.relaxed.gpu", "st.volatile", "st.weak", "st.cs", "stg128_coalesced",
                         "ld.relaxed.sys", "ldg.nc.u8"};
  for (int m = 0; m < 8; ++m) {
    for (int rep = 0; rep < 2; ++rep) {
      switch (m) {
        case 0: loop<0><<<1, 32>>>(buf, n, cyc, sink); break;
        case 1: loop<1><<<1, 32>>>(buf, n, cyc, sink); break;
        case 2: loop<2><<<1, 32>>>(buf, n, cyc, sink); break;
        case 3: loop<3><<<1, 32>>>(buf, n, cyc, sink); break;
        case 4: loop<4><<<1, 32>>>(buf, n, cyc, sink); break;
        case 5: loop<5><<<1, 32>>>(buf, n, cyc, sink); break;
        case 6: loop<6><<<1, 32>>>(buf, n, cyc, sink); break;
        case 7: loop<7><<<1, 32>>>(buf, n, cyc, sink); break;
      }
      cudaDeviceSynchronize();
    }
    long long h; cudaMemcpy(&h, cyc, 8, cudaMemcpyDeviceToHost);
    printf("%-18s %.1f cyc/iter\n", names[m], (double)h / n);
  }
  return 0;
}
