// mb10: issue cost (cycles per warp instruction) of the NW step's instruction classes on one
// SMSP: 8 independent chains per warp, 1 warp per SMSP (4 warps per CTA, 1 CTA).
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o mb10 mb10.cu && ./mb10
#include <cstdio>
#include <cstdint>

#define N 8
#define ITERS 4096

template <int OP>
__global__ void k(int32_t* out, long long* cyc, int32_t a0, int32_t g) {
  __shared__ int32_t sm[1024];
  for (int i = threadIdx.x; i < 1024; i += blockDim.x) sm[i] = i * 3;
  __syncthreads();
  int32_t v[N];
  for (int i = 0; i < N; ++i) v[i] = a0 + threadIdx.x * 7 + i;
  int32_t gg = g;
  asm volatile("mov.b32 %0, %0;" : "+r"(gg));
  __syncwarp();
  long long t0 = clock64();
#pragma unroll 1
  for (int it = 0; it < ITERS; ++it) {
#pragma unroll
    for (int r = 0; r < 8; ++r) {
#pragma unroll
      for (int i = 0; i < N; ++i) {
        if (OP == 0) v[i] = __viaddmax_s32(v[i], gg, v[(i + 1) % N]);           // VIADDMNMX
        if (OP == 1) v[i] = v[i] + v[(i + 1) % N];                              // IADD
        if (OP == 2) v[i] = max(v[i], v[(i + 1) % N]);                          // VIMNMX
        if (OP == 3) {                                                          // PRMT
          uint32_t r2;
          asm volatile("prmt.b32 %0, %1, %2, %3;" : "=r"(r2) : "r"(v[i]), "r"(gg), "r"(v[(i + 1) % N]));
          v[i] = r2;
        }
        if (OP == 4) v[i] = __shfl_sync(0xffffffffu, v[i], (threadIdx.x + 31) & 31);   // SHFL.IDX
        if (OP == 5) v[i] = __vimax3_s32(v[i], v[(i + 1) % N], gg);              // VIMNMX3
        if (OP == 6) v[i] = sm[(v[i] + i) & 1023];                               // LDS.32
        if (OP == 7) { sm[(threadIdx.x * 2 + i * 64 + r) & 1023] = v[i]; v[i] += 1; }   // STS.32 (+IADD)
        if (OP == 8) v[i] = (threadIdx.x & 31) == 31 ? gg : v[(i + 1) % N];    // SEL
        if (OP == 9) { int32_t a = v[i]; asm volatile("ld.shared.u16 %0, [%1];" : "=r"(a) : "r"((unsigned)__cvta_generic_to_shared(sm) + ((a + i) & 2046))); v[i] = a; }
        if (OP == 10) v[i] = __viaddmax_s32(v[i], gg, v[i]);                      // VIADDMNMX dependent chain (latency)
      }
    }
  }
  long long t1 = clock64();
  int32_t s = 0;
  for (int i = 0; i < N; ++i) s += v[i];
  out[blockIdx.x * blockDim.x + threadIdx.x] = s;
  if ((threadIdx.x & 31) == 0) cyc[threadIdx.x >> 5] = t1 - t0;
}

template <int OP>
void run(const char* name, int warps) {
  int32_t* o;
  long long* c;
  cudaMalloc(&o, 4096 * 4);
  cudaMalloc(&c, 64 * 8);
  k<OP><<<1, 32 * warps>>>(o, c, 1, -1);
  k<OP><<<1, 32 * warps>>>(o, c, 1, -1);
  long long h[64];
  cudaDeviceSynchronize();
  cudaMemcpy(h, c, warps * 8, cudaMemcpyDeviceToHost);
  double inst = double(ITERS) * 8 * N;
  printf("%-10s warps=%d cycles/warp-instr=%.2f\n", name, warps, h[0] / inst);
  cudaFree(o);
  cudaFree(c);
}

int main() {
  for (int w : {1, 4, 8}) {
    run<0>("VIADDMNMX", w);
    run<1>("IADD", w);
    run<2>("VIMNMX", w);
    run<3>("PRMT", w);
    run<4>("SHFL.IDX", w);
    run<5>("VIMNMX3", w);
    run<6>("LDS.32", w);
    run<7>("STS+IADD", w);
    run<8>("SEL", w);
    run<9>("LDS.U16", w);
  }
  return 0;
}
