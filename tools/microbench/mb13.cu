// mb13: cycles per step of the generation-8 NW lane pipeline in isolation (no memory, no
// barrier): which part of the ~50-cycle step is the shuffle chain and which is the cell.
//   v0  SHFL.IDX rotation + one VIADDMNMX                      (the lane-to-lane chain)
//   v1  the full K=2 step (scores, t, P, E, H), 1 warp
//   v2  v1 with 4 warps (one per SM sub-partition)
//   v3  v1 with SHFL.UP instead of the rotating SHFL.IDX
//   v4  v1, lane skew 2 (a lane's west input was produced two steps earlier)
#include <cstdio>
template <int V>
__global__ void kstep(int* out, int n, long long* cyc, unsigned seed) {
  const int lane = threadIdx.x & 31;
  const int srcl = (lane + 31) & 31;
  const bool is31 = lane == 31;
  const int g = -1, M = 1, X = -1;
  const int gLx = is31 ? -(1 << 29) : 2 * g;
  unsigned y0 = (seed >> lane) & 3, y1 = (seed >> (lane + 3)) & 3;
  int N0 = lane, N1 = lane + 1, NW = lane - 1, src = 0, q1 = 0;
  unsigned x = seed;
  long long t0 = clock64();
  for (int i = 0; i < n; ++i) {
#pragma unroll
    for (int u = 0; u < 16; ++u) {
      x = x * 1664525u + 1013904223u;   // row code stand-in (ALU, off the chain)
      const unsigned xc = (x >> 28) & 3;
      int W;
      if (V == 3) W = __shfl_up_sync(0xffffffffu, src, 1);
      else W = __shfl_sync(0xffffffffu, src, srcl);
      if (V == 4) { const int t = W; W = q1; q1 = t; }
      if (V == 0) {
        src = __viaddmax_s32(W, gLx, N0);
        continue;
      }
      const int s0 = xc == y0 ? M : X, s1 = xc == y1 ? M : X;
      const int t0_ = __viaddmax_s32(N0, g, NW + s0);
      const int t1_ = __viaddmax_s32(N1, g, N0 + s1);
      const int P1 = __viaddmax_s32(t0_, g, t1_);
      const int Px = is31 ? (int)(x & 7) : P1;
      src = __viaddmax_s32(W, gLx, Px);
      const int H0 = __viaddmax_s32(W, g, t0_);
      const int H1 = __viaddmax_s32(W, 2 * g, P1);
      NW = W;
      N0 = H0;
      N1 = H1;
    }
  }
  long long t1 = clock64();
  out[threadIdx.x] = N0 + N1 + src + NW;
  if (threadIdx.x == 0) *cyc = t1 - t0;
}
int main() {
  int* d;
  long long* c;
  cudaMalloc(&d, 4096);
  cudaMalloc(&c, 8);
  const int n = 4096;
  auto run = [&](auto k, int warps, const char* name) {
    k<<<1, 32 * warps>>>(d, n, c, 12345u);
    k<<<1, 32 * warps>>>(d, n, c, 12345u);
    long long h = 0;
    cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
    printf("%-40s %.2f cycles/step\n", name, double(h) / (16.0 * n));
  };
  run(kstep<0>, 1, "v0 shfl.idx + viaddmax chain, 1 warp");
  run(kstep<0>, 4, "v0 shfl.idx + viaddmax chain, 4 warps");
  run(kstep<1>, 1, "v1 full K=2 step, 1 warp");
  run(kstep<1>, 4, "v2 full K=2 step, 4 warps");
  run(kstep<3>, 1, "v3 full step, shfl.up, 1 warp");
  run(kstep<4>, 1, "v4 full step, skew 2, 1 warp");
  run(kstep<4>, 4, "v4 full step, skew 2, 4 warps");
  return 0;
}
