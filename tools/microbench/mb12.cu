// mb12: shared-window address of a kernel's dynamic shared memory (no static shared memory)
// -- decides whether the sweep's staging rings can be 32 KB-aligned by construction.
#include <cstdio>
extern "C" __global__ void probe(unsigned* out) {
  extern __shared__ __align__(1024) unsigned char raw[];
  if (threadIdx.x == 0) out[0] = static_cast<unsigned>(__cvta_generic_to_shared(raw));
}
int main() {
  unsigned* d;
  cudaMalloc(&d, 4);
  cudaFuncSetAttribute(probe, cudaFuncAttributeMaxDynamicSharedMemorySize, 200000);
  probe<<<1, 32, 200000>>>(d);
  unsigned h = 0;
  cudaMemcpy(&h, d, 4, cudaMemcpyDeviceToHost);
  int r = 0;
  cudaDeviceGetAttribute(&r, cudaDevAttrReservedSharedMemoryPerBlock, 0);
  printf("dynamic smem base 0x%x, reserved per block %d B\n", h, r);
  return 0;
}
