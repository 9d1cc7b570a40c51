// mb7: __nanosleep(t) actual duration on sm_100a (cycles via clock64, ns via globaltimer)
#include <cstdio>
__global__ void k(unsigned t, long long* out) {
  long long c0 = clock64();
  unsigned long long g0; asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(g0));
  for (int i = 0; i < 200; ++i) __nanosleep(t);
  long long c1 = clock64();
  unsigned long long g1; asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(g1));
  if (threadIdx.x == 0) { out[0] = (c1 - c0) / 200; out[1] = (long long)(g1 - g0) / 200; }
}
int main() {
  long long* d; cudaMalloc(&d, 16); long long h[2];
  unsigned ts[] = {0, 1, 8, 16, 32, 64, 100, 128, 200, 256, 500, 1000, 2000};
  for (unsigned t : ts) {
    for (int rep = 0; rep < 2; ++rep) { k<<<1, 32>>>(t, d); cudaMemcpy(h, d, 16, cudaMemcpyDeviceToHost); }
    printf("nanosleep(%u): %lld cycles, %lld ns per call\n", t, h[0], h[1]);
  }
}
