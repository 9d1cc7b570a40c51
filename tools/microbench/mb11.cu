// mb11: cost (cycles per occurrence, one warp) of the per-block synchronisation options of the
// NW sweep: after 32 STS.64 rows (a block), publish with
//   0 nothing, 1 __syncwarp, 2 fence.proxy.async.shared::cta + __syncwarp,
//   3 __threadfence_block (membar.cta), 4 __syncwarp + st.release.cta (lane 0),
//   5 mbarrier.arrive.release (all lanes), 6 __syncwarp + fence.acq_rel.cta (lane 0) + st
//   7 fence.proxy.async + TMA-free bulk commit (no copy)
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o mb11 mb11.cu && ./mb11
#include <cstdio>
#include <cstdint>

#define BLOCKS 2048

template <int OP>
__global__ void k(long long* cyc, int* out) {
  __shared__ __align__(16) int32_t st[32 * 2 * 64];
  __shared__ int flag;
  __shared__ __align__(8) unsigned long long mbar;
  const int lane = threadIdx.x & 31;
  if (threadIdx.x == 0) {
    flag = 0;
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"((unsigned)__cvta_generic_to_shared(&mbar)), "r"(1 << 20));
  }
  __syncthreads();
  int32_t a = lane, b = lane * 3;
  long long t0 = clock64();
#pragma unroll 1
  for (int blk = 0; blk < BLOCKS; ++blk) {
#pragma unroll
    for (int u = 0; u < 32; ++u) {
      a = __viaddmax_s32(a, b, u);
      *reinterpret_cast<int2*>(&st[((blk * 32 + u) & 63) * 64 + lane * 2]) = make_int2(a, b);
    }
    if (OP == 1) __syncwarp();
    if (OP == 2) {
      asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
      __syncwarp();
    }
    if (OP == 3) __threadfence_block();
    if (OP == 4) {
      __syncwarp();
      if (lane == 0)
        asm volatile("st.release.cta.shared.u32 [%0], %1;" ::"r"((unsigned)__cvta_generic_to_shared(&flag)), "r"(blk) : "memory");
    }
    if (OP == 5) {
      unsigned long long tok;
      asm volatile("mbarrier.arrive.release.cta.shared::cta.b64 %0, [%1];" : "=l"(tok) : "r"((unsigned)__cvta_generic_to_shared(&mbar)) : "memory");
      (void)tok;
    }
    if (OP == 6) {
      __syncwarp();
      if (lane == 0) {
        asm volatile("fence.acq_rel.cta;" ::: "memory");
        *reinterpret_cast<volatile int*>(&flag) = blk;
      }
    }
    if (OP == 7) {
      asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
      __syncwarp();
      if (lane == 0) *reinterpret_cast<volatile int*>(&flag) = blk;
    }
  }
  long long t1 = clock64();
  out[threadIdx.x] = a + st[lane];
  if (lane == 0) cyc[threadIdx.x >> 5] = t1 - t0;
}

template <int OP>
void run(const char* name) {
  long long* c;
  int* o;
  cudaMalloc(&c, 64 * 8);
  cudaMalloc(&o, 4096 * 4);
  k<OP><<<1, 32>>>(c, o);
  k<OP><<<1, 32>>>(c, o);
  long long h;
  cudaDeviceSynchronize();
  cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
  printf("%-34s cycles/block(32 steps)=%.1f\n", name, double(h) / BLOCKS);
  cudaFree(c);
  cudaFree(o);
}

int main() {
  run<0>("none");
  run<1>("syncwarp");
  run<2>("fence.proxy.async + syncwarp");
  run<3>("threadfence_block");
  run<4>("syncwarp + st.release.cta");
  run<5>("mbarrier.arrive.release (32 lanes)");
  run<6>("syncwarp + fence.acq_rel.cta + st");
  run<7>("fence.proxy.async + syncwarp + st");
  return 0;
}
