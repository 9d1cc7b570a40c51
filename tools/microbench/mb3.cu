// Core-loop microbenchmark of the NW lane pipeline (1 warp): cycles per row step for
// progressively richer bodies.  MODE bits: 1 = second (x) shuffle, 2 = STS.128 staging,
// 4 = PRMT score path, 8 = D=2 skew (use shuffle result two steps later).
#include <cstdio>
#include <cuda_runtime.h>

template <int MODE>
__global__ void core(int* out, int steps, long long* cyc, int g) {
  __shared__ int4 ring[64 * 32];
  const int lane = threadIdx.x;
  int Np[4] = {lane, lane + 1, lane + 2, lane + 3};
  int prevW = 0, q0 = 0, q1 = 0;
  unsigned xq0 = lane & 3, xq1 = 0;
  const unsigned qlo[4] = {0x01FF01FFu, 0xFF01FF01u, 0x0101FFFFu, 0xFFFF0101u};
  long long t0 = clock64();
#pragma unroll 4
  for (int t = 0; t < steps; ++t) {
    const int Win = (MODE & 8) ? q1 : q0;
    const unsigned X = (MODE & 8) ? xq1 : xq0;
    int H[4];
#pragma unroll
    for (int m = 0; m < 4; ++m) {
      const int NW = m == 0 ? prevW : Np[m - 1];
      const int W = m == 0 ? Win : H[m - 1];
      int s;
      if (MODE & 4) {
        unsigned r;
        asm("prmt.b32 %0, %1, %2, %3;" : "=r"(r) : "r"(qlo[m]), "r"(0u), "r"(X * 0x1111u + 0x8880u));
        s = (int)r;
      } else {
        s = (X == (unsigned)m) ? 1 : -1;
      }
      const int t1 = __viaddmax_s32(Np[m], g, NW + s);
      H[m] = __viaddmax_s32(W, g, t1);
    }
    prevW = Win;
#pragma unroll
    for (int m = 0; m < 4; ++m) Np[m] = H[m];
    if (MODE & 2) ring[((t & 63) * 32) + lane] = make_int4(H[0], H[1], H[2], H[3]);
    const int r = __shfl_up_sync(0xffffffffu, H[3], 1);
    q1 = q0;
    q0 = r;
    if (MODE & 1) {
      const unsigned xs = __shfl_up_sync(0xffffffffu, X, 1);
      xq1 = xq0;
      xq0 = xs;
    }
  }
  long long t1c = clock64();
  out[lane] = Np[0] + Np[3] + (int)xq0 + ring[lane].x;
  if (lane == 0) *cyc = t1c - t0;
}

int main() {
  int* o; long long* c; cudaMalloc(&o, 4096); cudaMalloc(&c, 8);
  const int steps = 40000;
  auto run = [&](auto kern, const char* name) {
    kern<<<1, 32>>>(o, steps, c, -1); cudaDeviceSynchronize();
    kern<<<1, 32>>>(o, steps, c, -1); cudaDeviceSynchronize();
    long long h; cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
    printf("%-28s %.1f cyc/step\n", name, (double)h / steps);
  };
  run(core<0>, "cells+1shfl");
  run(core<1>, "+xshfl");
  run(core<2>, "+STS.128");
  run(core<3>, "+xshfl+STS");
  run(core<7>, "+xshfl+STS+PRMT");
  run(core<8>, "D2 cells+1shfl");
  run(core<15>, "D2 all");
  return 0;
}
