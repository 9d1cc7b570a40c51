// mb9: candidate n=16 Nash solvers -- correctness vs the current nash_solve16 on random keys,
// then latency (1 warp/SM) and throughput (28 warps/SM) of key chain + solver.
#include <cstdio>
#include "../../paper_conf_ppopp_mohantyc14_b200/csrc/wf_nash.cuh"
using namespace wfk;

// Row/column ownership: lane l < 16 owns row a = l of B, lane 16 + b owns column b of A.
__device__ __forceinline__ void solve_rc(uint32_t key, int lane, uint32_t o[4]) {
  const bool isB = lane < 16;
  const uint32_t t0 = static_cast<uint32_t>(lane & 15);
  // entry idx = 16a + b; hash input c = 2 idx (+1 for B), c < 2^16: first xorshift folds
  const uint32_t K1 = key ^ (key >> 16);
  const uint32_t KL = K1 ^ (isB ? (32u * t0 + 1u) : (2u * t0));
  const uint32_t sh = isB ? 1u : 5u;
  uint32_t v[16];
#pragma unroll
  for (int t = 0; t < 16; ++t) v[t] = lowbias32_tail_byte(KL ^ (static_cast<uint32_t>(t) << sh));
  uint32_t mx = v[0];
#pragma unroll
  for (int t = 1; t < 16; ++t) mx = max(mx, v[t]);
  uint32_t mask = 0;
#pragma unroll
  for (int t = 0; t < 16; ++t) mask |= (v[t] == mx) ? (1u << t) : 0u;
  // transpose the A masks (lanes 16..31, row = column b, bit = a) into lanes 0..15 (row a, bit b)
  uint32_t x = mask;
  {
    auto step = [&](int s, uint32_t m) {
      const uint32_t y = __shfl_xor_sync(0xffffffffu, x, s);
      const uint32_t up = (x & m) | ((y << s) & ~m);          // lane bit s clear: keep low, take partner low
      const uint32_t dn = (x & ~m) | ((y >> s) & m);          // lane bit s set: keep high, take partner high
      x = (lane & s) ? dn : up;
    };
    step(8, 0x00FF00FFu);
    step(4, 0x0F0F0F0Fu);
    step(2, 0x33333333u);
    step(1, 0x55555555u);
  }
  const uint32_t AT = __shfl_xor_sync(0xffffffffu, x, 16);
  const uint32_t ne = isB ? (mask & AT) : 0u;
  const int count = static_cast<int>(__reduce_add_sync(0xffffffffu, __popc(ne)));
  const uint32_t myfirst = ne ? 16u * t0 + (__ffs(ne) - 1) : 0xFFFFu;
  const uint32_t f = __reduce_min_sync(0xffffffffu, myfirst);
  // at an equilibrium A equals its column maximum and B its row maximum
  const uint32_t pa = __shfl_sync(0xffffffffu, mx, 16 + (f & 15));
  const uint32_t pb = __shfl_sync(0xffffffffu, mx, (f >> 4) & 15);
  const bool none = f == 0xFFFFu;
  o[0] = static_cast<uint32_t>(count);
  o[1] = none ? 0xFFFFFFFFu : f;
  o[2] = none ? 0xFFFFFFFFu : pa;
  o[3] = none ? 0xFFFFFFFFu : pb;
}

__global__ void check(int nkeys, int* bad, uint32_t* hist) {
  const int lane = threadIdx.x & 31;
  for (int i = blockIdx.x * (blockDim.x / 32) + threadIdx.x / 32; i < nkeys; i += gridDim.x * (blockDim.x / 32)) {
    const uint32_t key = lowbias32(0x1234567u + 7919u * i);
    uint32_t a[4], b[4];
    nash_solve16(key, lane, a);
    solve_rc(key, lane, b);
    if (lane == 0) {
      for (int p = 0; p < 4; ++p) if (a[p] != b[p]) atomicAdd(bad, 1);
      atomicAdd(hist + min(a[0], 7u), 1u);
    }
  }
}

template <int V>
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
#pragma unroll
    for (int p = 0; p < 4; ++p) key = lowbias32(key ^ W[p]);
    uint32_t o[4];
    if (V == 0) nash_solve16(key, lane, o); else solve_rc(key, lane, o);
#pragma unroll
    for (int p = 0; p < 4; ++p) { NW[p] = W[p]; W[p] = N[p]; N[p] = o[p]; }
  }
  long long t1 = clock64();
  if (lane == 0) { out[blockIdx.x * 32 + (threadIdx.x >> 5)] = N[0] ^ N[1]; if (threadIdx.x == 0 && blockIdx.x == 0) *cyc = (t1 - t0); }
}
int main() {
  int* bad; uint32_t* hist; cudaMalloc(&bad, 4); cudaMalloc(&hist, 32); cudaMemset(bad, 0, 4); cudaMemset(hist, 0, 32);
  const int nkeys = 1 << 20;
  check<<<592, 256>>>(nkeys, bad, hist);
  int hb; uint32_t hh[8]; cudaMemcpy(&hb, bad, 4, cudaMemcpyDeviceToHost); cudaMemcpy(hh, hist, 32, cudaMemcpyDeviceToHost);
  printf("check: %d mismatching words over %d keys; NE-count histogram 0..7+: %u %u %u %u %u %u %u %u\n", hb, nkeys,
         hh[0], hh[1], hh[2], hh[3], hh[4], hh[5], hh[6], hh[7]);
  unsigned* o; long long* c; cudaMalloc(&o, 1 << 20); cudaMalloc(&c, 8);
  for (int v = 0; v < 2; ++v)
    for (int w : {1, 8, 28}) {
      long long h; const int iters = 2000;
      auto kf = v == 0 ? k<0> : k<1>;
      kf<<<148, 32 * w>>>(iters, o, c); cudaDeviceSynchronize();
      kf<<<148, 32 * w>>>(iters, o, c); cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
      printf("%s warps/SM=%2d: %.0f cycles per cell per warp, %.1f per cell per SM\n", v ? "rowcol " : "current", w,
             (double)h / iters, (double)h / iters / w);
    }
}
