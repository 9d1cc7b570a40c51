// mb8: latency / throughput of one Nash cell (key chain + nash_solve16) on sm_100a.
// W warps per CTA, 1 CTA per SM; each warp runs `iters` dependent cells (N = previous output).
#include <cstdio>
#include "../../paper_conf_ppopp_mohantyc14_b200/csrc/wf_nash.cuh"
using namespace wfk;
__global__ void k(int iters, unsigned* out, long long* cyc) {
  const int lane = threadIdx.x & 31;
  uint32_t N[4] = {threadIdx.x, 2, 3, 4}, NW[4] = {5, 6, 7, 8}, W[4] = {9, 10, 11, 12};
  long long t0 = clock64();
  for (int it = 0; it < iters; ++it) {
    uint32_t key = kNashSeed;
#pragma unroll
    for (int p = 0; p < 4; ++p) key = lowbias32(key ^ N[p]);
#pragma unroll
    for (int p = 0; p < 4; ++p) key = lowbias32(key ^ NW[p]);
    key = lowbias32(key ^ (uint32_t)it);
    key = lowbias32(key ^ 77u);
#ifndef PREFIX_ONLY
#pragma unroll
    for (int p = 0; p < 4; ++p) key = lowbias32(key ^ W[p]);
    uint32_t o[4];
    nash_solve16(key, lane, o);
#else
    uint32_t o[4] = {key, key + 1, key + 2, key + 3};
#endif
#pragma unroll
    for (int p = 0; p < 4; ++p) { NW[p] = W[p]; W[p] = N[p]; N[p] = o[p]; }
  }
  long long t1 = clock64();
  if (lane == 0) { out[blockIdx.x * 32 + (threadIdx.x >> 5)] = N[0] ^ N[1]; if (threadIdx.x == 0 && blockIdx.x == 0) *cyc = (t1 - t0); }
}
int main() {
  unsigned* o; long long* c; cudaMalloc(&o, 1 << 20); cudaMalloc(&c, 8);
  for (int w : {1, 2, 4, 8, 16, 28}) {
    long long h; const int iters = 2000;
    k<<<148, 32 * w>>>(iters, o, c); cudaDeviceSynchronize();
    k<<<148, 32 * w>>>(iters, o, c); cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
    printf("warps/SM=%2d: %.0f cycles per cell per warp, %.1f cycles per cell per SM\n", w, (double)h / iters, (double)h / iters / w);
  }
}
