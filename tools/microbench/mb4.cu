// Core of a "KR x KC register tile per lane" NW pipeline (1 warp): cycles per step, where a
// step computes a KR-row x KC-column tile per lane and passes the east column (KR values)
// and the packed row codes to the next lane by shuffle.
#include <cstdio>
#include <cuda_runtime.h>

__device__ __forceinline__ int prmt_s8(unsigned lo, unsigned sel) {
  unsigned r;
  asm("prmt.b32 %0, %1, %2, %3;" : "=r"(r) : "r"(lo), "r"(0u), "r"(sel));
  return (int)r;
}

template <int KR, int KC, bool STS>
__global__ void core(int* out, int steps, long long* cyc, int g) {
  __shared__ int4 ring[80 * 32];
  const int lane = threadIdx.x;
  int Np[KC];
  unsigned q[KC];
#pragma unroll
  for (int m = 0; m < KC; ++m) { Np[m] = lane + m; q[m] = 0x01FF01FFu ^ (m * 0x01010101u); }
  int prevW = 0;
  int Wq[KR];
#pragma unroll
  for (int i = 0; i < KR; ++i) Wq[i] = i;
  unsigned Xq = 0x03020100u ^ lane;
  int slot = 0;
  long long t0 = clock64();
  for (int t = 0; t < steps; ++t) {
    int H[KR][KC];
#pragma unroll
    for (int i = 0; i < KR; ++i) {
      const unsigned x = (Xq >> (8 * i)) & 0xFFu;
      const unsigned sel = x * 0x1111u + 0x8880u;
#pragma unroll
      for (int m = 0; m < KC; ++m) {
        const int N = i == 0 ? Np[m] : H[i - 1][m];
        const int NW = m == 0 ? (i == 0 ? prevW : Wq[i - 1]) : (i == 0 ? Np[m - 1] : H[i - 1][m - 1]);
        const int W = m == 0 ? Wq[i] : H[i][m - 1];
        const int s = prmt_s8(q[m], sel);
        const int t1 = __viaddmax_s32(N, g, NW + s);
        H[i][m] = __viaddmax_s32(W, g, t1);
      }
    }
    prevW = Wq[KR - 1];
#pragma unroll
    for (int m = 0; m < KC; ++m) Np[m] = H[KR - 1][m];
    if (STS) {
#pragma unroll
      for (int i = 0; i < KR; ++i) {
        if (KC == 4) ring[((slot + i) % 80) * 32 + lane] = make_int4(H[i][0], H[i][1], H[i][2], H[i][3]);
      }
      slot = (slot + KR) % 80;
    }
#pragma unroll
    for (int i = 0; i < KR; ++i) Wq[i] = __shfl_up_sync(0xffffffffu, H[i][KC - 1], 1);
    Xq = __shfl_up_sync(0xffffffffu, Xq, 1);
  }
  long long t1c = clock64();
  int acc = Np[0] + (int)Xq;
#pragma unroll
  for (int i = 0; i < KR; ++i) acc += Wq[i];
  out[lane] = acc + ((int*)ring)[lane];
  if (lane == 0) *cyc = t1c - t0;
}

int main() {
  int* o; long long* c; cudaMalloc(&o, 4096); cudaMalloc(&c, 8);
  const int steps = 20000;
  auto run = [&](auto kern, const char* name, int cells) {
    kern<<<1, 32>>>(o, steps, c, -1); cudaDeviceSynchronize();
    kern<<<1, 32>>>(o, steps, c, -1); cudaDeviceSynchronize();
    long long h; cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
    printf("%-20s %.1f cyc/step  %.2f cyc/cell/lane\n", name, (double)h / steps, (double)h / steps / cells);
  };
  run(core<4, 4, false>, "4x4 noSTS", 16);
  run(core<4, 4, true>, "4x4 STS", 16);
  run(core<2, 4, true>, "2x4 STS", 8);
  run(core<8, 4, true>, "8x4 STS", 32);
  run(core<1, 4, true>, "1x4 STS", 4);
  return 0;
}
