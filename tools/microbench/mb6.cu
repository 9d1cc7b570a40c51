// Times the production NwWarp<K,1,1,16,PRMT>::block<false> steady body in isolation:
// warp 0 runs B blocks; optionally warp 1 runs an I/O-like polling loop (LDS + ballot +
// STS + nanosleep) on the same SM to measure MIO interference.
#include <cstdio>
#include "../../paper_conf_ppopp_mohantyc14_b200/csrc/wf_nw.cuh"

using namespace wfk;

template <int K, bool POLLER>
__global__ void bench(SweepLaunch L, int blocks, long long* cyc, int* out) {
  constexpr int U = 16;
  using S = NwSmem<K, 1, 1, U>;
  extern __shared__ __align__(16) unsigned char raw[];
  const S sm(raw);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  __shared__ volatile int stop;
  if (threadIdx.x == 0) stop = 0;
  __syncthreads();
  if (warp == 0) {
    NwWarp<K, 1, 1, U, true> w(L, nullptr, sm, 0, 0, lane);
    uint32_t xc[U];
    for (int u = 0; u < U; ++u) xc[u] = (lane + u) & 3;
    int32_t east[U];
    long long t0 = clock64();
    int t = 64;
    for (int b = 0; b < blocks; ++b, t += U) w.template block<false>(t, lane * 3, xc, east);
    long long t1 = clock64();
    if (lane == 0) { *cyc = t1 - t0; stop = 1; }
    out[lane] = east[U - 1] + w.Np[0];
  } else if (POLLER) {
    int acc = 0;
    while (!stop) {
      const unsigned long long v = lds_vol(sm.hand_slot(1, lane));
      acc += (int)__ballot_sync(0xffffffffu, (v >> 32) == 7u);
      sts_vol_i(sm.prog + 1, acc);
      __nanosleep(100);
    }
    out[32 + lane] = acc;
  }
}

int main() {
  SweepLaunch L{};
  L.rows = 1 << 20; L.c0 = 0; L.c1 = 1 << 20; L.band_w = 128; L.nbands = 1; L.gap = -1; L.match = 1; L.mismatch = -1;
  unsigned char* y; cudaMalloc(&y, 1 << 20); cudaMemset(y, 1, 1 << 20); L.col_in = y;
  long long* c; int* o; cudaMalloc(&c, 8); cudaMalloc(&o, 1024);
  const int blocks = 4000;
  auto run = [&](auto kern, int nthreads, size_t smem, const char* name) {
    cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    kern<<<1, nthreads, smem>>>(L, blocks, c, o); cudaDeviceSynchronize();
    kern<<<1, nthreads, smem>>>(L, blocks, c, o);
    cudaError_t e = cudaDeviceSynchronize();
    long long h; cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
    printf("%-26s %s %.1f cyc/step\n", name, cudaGetErrorString(e), (double)h / blocks / 16);
  };
  run(bench<4, false>, 32, NwSmem<4, 1, 1, 16>::bytes, "K4 block<false> alone");
  run(bench<4, true>, 64, NwSmem<4, 1, 1, 16>::bytes, "K4 block<false> + poller");
  run(bench<2, false>, 32, NwSmem<2, 1, 1, 16>::bytes, "K2 block<false> alone");
  return 0;
}
