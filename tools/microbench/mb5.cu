// NW lane-pipeline core with the prefix-max cell (W enters through ONE op per cell):
//   t1[m] = max(N[m] + g, NW[m] + s[m]);  P[m] = max(t1[m], P[m-1] + g);
//   H[m]  = max(P[m], W + (m+1) g)
// and the row codes pipelined two steps ahead.  cycles per row step, 1 warp.
#include <cstdio>
#include <cuda_runtime.h>

__device__ __forceinline__ int prmt_s8(unsigned lo, unsigned sel) {
  unsigned r;
  asm("prmt.b32 %0, %1, %2, %3;" : "=r"(r) : "r"(lo), "r"(0u), "r"(sel));
  return (int)r;
}

template <int K, int D, bool PREFIX>
__global__ void core(int* out, int steps, long long* cyc, int g) {
  __shared__ int4 ring[32 * 32 * (K / 4)];
  const int lane = threadIdx.x;
  int Np[K];
  unsigned q[K];
  int gk[K];
#pragma unroll
  for (int m = 0; m < K; ++m) { Np[m] = lane + m; q[m] = 0x01FF01FFu ^ (m * 0x01010101u); gk[m] = (m + 1) * g; }
  int prevW = 0;
  int Wq[D];
#pragma unroll
  for (int d = 0; d < D; ++d) Wq[d] = d;
  unsigned x0 = lane & 3, x1 = (lane + 1) & 3;
  long long t0 = clock64();
#pragma unroll 4
  for (int t = 0; t < steps; ++t) {
    const int W = Wq[D - 1];
    const unsigned sel = x0 * 0x1111u + 0x8880u;
    int H[K];
    if (PREFIX) {
      int P = 0;
#pragma unroll
      for (int m = 0; m < K; ++m) {
        const int NW = m == 0 ? prevW : Np[m - 1];
        const int t1 = __viaddmax_s32(Np[m], g, NW + prmt_s8(q[m], sel));
        P = m == 0 ? t1 : __viaddmax_s32(P, g, t1);
        H[m] = __viaddmax_s32(W, gk[m], P);
      }
    } else {
#pragma unroll
      for (int m = 0; m < K; ++m) {
        const int NW = m == 0 ? prevW : Np[m - 1];
        const int t1 = __viaddmax_s32(Np[m], g, NW + prmt_s8(q[m], sel));
        H[m] = __viaddmax_s32(m == 0 ? W : H[m - 1], g, t1);
      }
    }
    prevW = W;
#pragma unroll
    for (int m = 0; m < K; ++m) Np[m] = H[m];
#pragma unroll
    for (int k = 0; k < K / 4; ++k)
      ring[((t & 31) * 32 + lane) * (K / 4) + k] = make_int4(H[4 * k], H[4 * k + 1], H[4 * k + 2], H[4 * k + 3]);
    const int r = __shfl_up_sync(0xffffffffu, H[K - 1], 1);
    const unsigned xs = __shfl_up_sync(0xffffffffu, x1, 1);   // lane-1's NEXT code = my code two steps on
#pragma unroll
    for (int d = D - 1; d > 0; --d) Wq[d] = Wq[d - 1];
    Wq[0] = r;
    x0 = x1;
    x1 = xs;
  }
  long long t1c = clock64();
  out[lane] = Np[0] + Np[K - 1] + (int)x0 + ((int*)ring)[lane];
  if (lane == 0) *cyc = t1c - t0;
}

int main() {
  int* o; long long* c; cudaMalloc(&o, 4096); cudaMalloc(&c, 8);
  const int steps = 40000;
  auto run = [&](auto kern, const char* name) {
    kern<<<1, 32>>>(o, steps, c, -1); cudaDeviceSynchronize();
    kern<<<1, 32>>>(o, steps, c, -1); cudaDeviceSynchronize();
    long long h; cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
    printf("%-24s %.1f cyc/step\n", name, (double)h / steps);
  };
  run(core<4, 1, false>, "K4 D1 chain");
  run(core<4, 1, true>, "K4 D1 prefix");
  run(core<4, 2, true>, "K4 D2 prefix");
  run(core<8, 1, true>, "K8 D1 prefix");
  run(core<8, 1, false>, "K8 D1 chain");
  run(core<8, 2, true>, "K8 D2 prefix");
  return 0;
}
