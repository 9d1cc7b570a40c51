// mb14: cycles per lane-pipeline step of candidate NW cell formulations (round 2, generation-8
// successor study), with the per-step shared-memory traffic of the real kernel (x code LDS,
// staging STS, lane-31 east STS, per-block ring LDS.128 + named CTA barrier).  4 warps, one per
// SM sub-partition.
//   K    columns per lane (2, 4)
//   FORM 0 prefix (generation 8: t, P, H per cell, E on the chain after one op)
//        1 direct (t, H = max(t, H_{m-1} + g); chain K ops)
//        2 mixed  (P prefix only for the east column: src after one op; H direct off the chain)
//   SC   0 ISETP + SEL scores, 1 PRMT byte lookup (alphabet <= 8; row selector by IMAD)
//   MEM  0 registers only, 1 with the kernel's shared-memory traffic
#include <cstdio>
#include <cstdint>

constexpr unsigned FULL = 0xffffffffu;

__device__ __forceinline__ int vmax(int a, int b, int c) { return __viaddmax_s32(a, b, c); }
__device__ __forceinline__ int prmt(unsigned a, unsigned b, unsigned s) {
  unsigned d;
  asm("prmt.b32 %0, %1, %2, %3;" : "=r"(d) : "r"(a), "r"(b), "r"(s));
  return (int)d;
}

template <int K, int FORM, int SC, int MEM>
__global__ void __launch_bounds__(128, 1) kstep(int* out, int nblk, long long* cyc, unsigned seed) {
  __shared__ __align__(16) unsigned char xs[4096];
  __shared__ __align__(16) int stage[4][16][32 * K];
  __shared__ __align__(16) int ring[5][128];
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  for (int i = threadIdx.x; i < 4096; i += blockDim.x) xs[i] = (unsigned char)((i * 2654435761u + seed) >> 29) & 3;
  for (int i = threadIdx.x; i < 5 * 128; i += blockDim.x) (&ring[0][0])[i] = i;
  __syncthreads();
  const int srcl = (lane + 31) & 31;
  const bool is31 = lane == 31;
  const int g = -1, M = 1, X = -1;
  const int gLx = is31 ? -(1 << 29) : (FORM == 1 ? g : K * g);
  unsigned y[K];
  unsigned tab_lo[K], tab_hi[K];
  int N[K], gk[K];
#pragma unroll
  for (int m = 0; m < K; ++m) {
    y[m] = (seed >> (lane + 3 * m)) & 3;
    N[m] = lane * K + m;
    gk[m] = (m + 1) * g;
    unsigned lo = 0, hi = 0;
#pragma unroll
    for (int c = 0; c < 4; ++c) lo |= (unsigned)((c == (int)y[m] ? M : X) & 255) << (8 * c);
    tab_lo[m] = lo;
    tab_hi[m] = hi;
  }
  int NWc = lane * K - 1, src = 0;
  const uint32_t xb = (uint32_t)__cvta_generic_to_shared(xs);
  const uint32_t sb = (uint32_t)__cvta_generic_to_shared(&stage[warp][0][0]) + lane * 4 * K;
  const uint32_t rin = (uint32_t)__cvta_generic_to_shared(&ring[warp][0]);
  const uint32_t rout = (uint32_t)__cvta_generic_to_shared(&ring[warp + 1][0]);
  long long t0 = clock64();
  int s = 0;
  unsigned xq[16];   // x codes of the current block, loaded one block ahead (as the kernel does)
#pragma unroll
  for (int u = 0; u < 16; ++u) xq[u] = xs[(u - lane) & 4095];
  for (int b = 0; b < nblk; ++b) {
    int in[16];
    if (MEM) {
#pragma unroll
      for (int q = 0; q < 4; ++q) {
        int4 v;
        asm volatile("ld.shared.v4.s32 {%0,%1,%2,%3}, [%4];" : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "r"(rin + 64 * q + 16 * (b & 1)));
        in[4 * q] = v.x; in[4 * q + 1] = v.y; in[4 * q + 2] = v.z; in[4 * q + 3] = v.w;
      }
    } else {
#pragma unroll
      for (int u = 0; u < 16; ++u) in[u] = b + u;
    }
#pragma unroll
    for (int u = 0; u < 16; ++u, ++s) {
      unsigned xc;
      if (MEM) {
        xc = xq[u];
        xq[u] = xs[(s + 16 - lane) & 4095];
      } else {
        xc = ((unsigned)(s * 2654435761u) >> 30);
      }
      const int W = __shfl_sync(FULL, src, srcl);
      int t[K], Hv[K], sc[K];
      unsigned sel = 0;
      if (SC == 1) sel = xc * 0x1111u + 0x8880u;
#pragma unroll
      for (int m = 0; m < K; ++m) {
        sc[m] = SC == 1 ? prmt(tab_lo[m], tab_hi[m], sel) : (xc == y[m] ? M : X);
        const int nw = m == 0 ? NWc : N[m - 1];
        t[m] = vmax(N[m], g, nw + sc[m]);
      }
      if (FORM == 0) {
        int P[K];
        P[0] = t[0];
#pragma unroll
        for (int m = 1; m < K; ++m) P[m] = vmax(P[m - 1], g, t[m]);
        const int Px = is31 ? in[u] : P[K - 1];
        src = vmax(W, gLx, Px);
#pragma unroll
        for (int m = 0; m < K; ++m) Hv[m] = vmax(W, gk[m], P[m]);
      } else if (FORM == 1) {
        Hv[0] = vmax(W, g, t[0]);
#pragma unroll
        for (int m = 1; m < K - 1; ++m) Hv[m] = vmax(Hv[m - 1], g, t[m]);
        const int Tx = is31 ? in[u] : t[K - 1];
        src = vmax(Hv[K - 2], gLx, Tx);
        Hv[K - 1] = vmax(Hv[K - 2], g, t[K - 1]);
      } else {
        int P = t[0];
#pragma unroll
        for (int m = 1; m < K; ++m) P = vmax(P, g, t[m]);
        const int Px = is31 ? in[u] : P;
        src = vmax(W, gLx, Px);
        Hv[0] = vmax(W, g, t[0]);
#pragma unroll
        for (int m = 1; m < K; ++m) Hv[m] = vmax(Hv[m - 1], g, t[m]);
      }
      if (MEM) {
        int* a = &stage[warp][(s - lane) & 15][lane * K];
        if (K == 2) *reinterpret_cast<int2*>(a) = make_int2(Hv[0], Hv[1]);
        else *reinterpret_cast<int4*>(a) = make_int4(Hv[0], Hv[1], Hv[2], Hv[K - 1]);
        if (is31) ring[warp + 1][(s + 2) & 127] = Hv[K - 1];
      }
      NWc = W;
#pragma unroll
      for (int m = 0; m < K; ++m) N[m] = Hv[m];
    }
    if (MEM) asm volatile("bar.sync 1, 128;" ::: "memory");
  }
  long long t1 = clock64();
  int acc = src + NWc;
#pragma unroll
  for (int m = 0; m < K; ++m) acc += N[m];
  out[threadIdx.x] = acc;
  if (threadIdx.x == 0) *cyc = t1 - t0;
}


// H = 2 rows per step, K = 2.  FORM 0: prefix form per row, row 1's east after a SEL on the chain
// (generation 9 as built); FORM 1: row 1's east in max-plus form (two ops after W).
template <int FORM, int MEM>
__global__ void __launch_bounds__(128, 1) kstep2(int* out, int nblk, long long* cyc, unsigned seed) {
  constexpr int K = 2;
  __shared__ __align__(16) unsigned char xs[4096];
  __shared__ __align__(16) int stage[4][16][32 * K];
  __shared__ __align__(16) int ring[5][128];
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  for (int i = threadIdx.x; i < 4096; i += blockDim.x) xs[i] = (unsigned char)((i * 2654435761u + seed) >> 29) & 3;
  for (int i = threadIdx.x; i < 5 * 128; i += blockDim.x) (&ring[0][0])[i] = i;
  __syncthreads();
  const int srcl = (lane + 31) & 31;
  const bool is31 = lane == 31;
  const int g = -1, M = 1, X = -1;
  const int gLx = is31 ? -(1 << 29) : K * g;
  unsigned y0 = (seed >> lane) & 3, y1 = (seed >> (lane + 3)) & 3;
  int N0 = lane * K, N1 = lane * K + 1;
  // row-1 max-plus constants: c_m = max((m+2)g, m g + s)
  const int c0M = max(2 * g, M), c0X = max(2 * g, X), c1M = max(3 * g, g + M), c1X = max(3 * g, g + X);
  int NWc = lane * K - 1, src0 = 0, src1 = 0;
  const uint32_t rin = (uint32_t)__cvta_generic_to_shared(&ring[warp][0]);
  long long t0 = clock64();
  int s = 0;
  unsigned xq[16];
#pragma unroll
  for (int u = 0; u < 16; ++u) xq[u] = xs[(u - 2 * lane) & 4095];
  for (int b = 0; b < nblk; ++b) {
    int in[16];
    if (MEM) {
#pragma unroll
      for (int q = 0; q < 4; ++q) {
        int4 v;
        asm volatile("ld.shared.v4.s32 {%0,%1,%2,%3}, [%4];" : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "r"(rin + 64 * q + 16 * (b & 1)));
        in[4 * q] = v.x; in[4 * q + 1] = v.y; in[4 * q + 2] = v.z; in[4 * q + 3] = v.w;
      }
    } else {
#pragma unroll
      for (int u = 0; u < 16; ++u) in[u] = b + u;
    }
#pragma unroll
    for (int u = 0; u < 8; ++u, ++s) {
      unsigned xa, xb2;
      if (MEM) {
        xa = xq[2 * u]; xb2 = xq[2 * u + 1];
        xq[2 * u] = xs[(2 * s + 16 - 2 * lane) & 4095];
        xq[2 * u + 1] = xs[(2 * s + 17 - 2 * lane) & 4095];
      } else {
        xa = ((unsigned)(s * 2654435761u) >> 30); xb2 = ((unsigned)(s * 2246822519u) >> 30);
      }
      const int W0 = __shfl_sync(FULL, src0, srcl);
      const int W1 = __shfl_sync(FULL, src1, srcl);
      // row 0
      const bool e00 = xa == y0, e01 = xa == y1;
      const int t00 = vmax(N0, g, NWc + (e00 ? M : X));
      const int t01 = vmax(N1, g, N0 + (e01 ? M : X));
      const int P01 = vmax(t00, g, t01);
      src0 = vmax(W0, gLx, is31 ? in[2 * u] : P01);
      const int H00 = vmax(W0, g, t00), H01 = vmax(W0, 2 * g, P01);
      const bool e10 = xb2 == y0, e11 = xb2 == y1;
      int H10, H11;
      if (FORM == 0) {
        const int t10 = vmax(H00, g, W0 + (e10 ? M : X));
        const int t11 = vmax(H01, g, H00 + (e11 ? M : X));
        const int P11 = vmax(t10, g, t11);
        src1 = vmax(W1, gLx, is31 ? in[2 * u + 1] : P11);
        H10 = vmax(W1, g, t10);
        H11 = vmax(W1, 2 * g, P11);
      } else {
        // t1_m = max(T_m, W0 + c_m); P1_m = max(TP_m, W0 + CP_m); H1_m = max(P1_m, W1 + (m+1)g)
        const int T0 = t00 + g;
        const int T1 = vmax(P01, g, t00 + (e11 ? M : X));
        const int c0 = e10 ? c0M : c0X, c1 = e11 ? c1M : c1X;
        const int TP1 = vmax(T0, g, T1), CP1 = vmax(c0, g, c1);
        const int P10 = vmax(W0, c0, T0);
        const int P11 = vmax(W0, CP1, TP1);
        const int Px = vmax(W0, is31 ? -(1 << 29) : CP1, is31 ? in[2 * u + 1] : TP1);
        src1 = vmax(W1, gLx, Px);
        H10 = vmax(W1, g, P10);
        H11 = vmax(W1, 2 * g, P11);
      }
      if (MEM) {
        *reinterpret_cast<int2*>(&stage[warp][(2 * s - 2 * lane) & 15][lane * K]) = make_int2(H00, H01);
        *reinterpret_cast<int2*>(&stage[warp][(2 * s + 1 - 2 * lane) & 15][lane * K]) = make_int2(H10, H11);
        if (is31) *reinterpret_cast<int2*>(&ring[warp + 1][(2 * s + 2) & 127]) = make_int2(H01, H11);
      }
      NWc = W1;
      N0 = H10;
      N1 = H11;
    }
    if (MEM) asm volatile("bar.sync 1, 128;" ::: "memory");
  }
  long long t1 = clock64();
  out[threadIdx.x] = src0 + src1 + NWc + N0 + N1;
  if (threadIdx.x == 0) *cyc = t1 - t0;
}

int main() {
  int* d;
  long long* c;
  cudaMalloc(&d, 4096);
  cudaMalloc(&c, 8);
  const int nblk = 2048;
  auto run = [&](auto k, const char* name, int K) {
    k<<<1, 128>>>(d, nblk, c, 12345u);
    k<<<1, 128>>>(d, nblk, c, 12345u);
    cudaError_t e = cudaDeviceSynchronize();
    long long h = 0;
    cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
    const double cps = double(h) / (16.0 * nblk);
    printf("%-34s %6.2f cycles/step  %5.2f cycles/column  %s\n", name, cps, cps / K, e ? cudaGetErrorString(e) : "");
  };
  {
    auto run2 = [&](auto k, const char* name) {
      k<<<1, 128>>>(d, nblk, c, 12345u);
      k<<<1, 128>>>(d, nblk, c, 12345u);
      cudaDeviceSynchronize();
      long long h = 0;
      cudaMemcpy(&h, c, 8, cudaMemcpyDeviceToHost);
      const double cps = double(h) / (8.0 * nblk);
      printf("%-34s %6.2f cycles/step  %5.2f cycles/row\n", name, cps, cps / 2);
    };
    run2(kstep2<0, 0>, "H2K2 as built      reg");
    run2(kstep2<0, 1>, "H2K2 as built      mem");
    run2(kstep2<1, 0>, "H2K2 max-plus row1 reg");
    run2(kstep2<1, 1>, "H2K2 max-plus row1 mem");
  }
  run(kstep<2, 0, 0, 0>, "K2 prefix  isetp  reg", 2);
  run(kstep<2, 0, 0, 1>, "K2 prefix  isetp  mem", 2);
  run(kstep<2, 0, 1, 1>, "K2 prefix  prmt   mem", 2);
  run(kstep<2, 1, 0, 1>, "K2 direct  isetp  mem", 2);
  run(kstep<2, 1, 1, 1>, "K2 direct  prmt   mem", 2);
  run(kstep<2, 2, 1, 1>, "K2 mixed   prmt   mem", 2);
  run(kstep<4, 0, 0, 0>, "K4 prefix  isetp  reg", 4);
  run(kstep<4, 0, 0, 1>, "K4 prefix  isetp  mem", 4);
  run(kstep<4, 0, 1, 1>, "K4 prefix  prmt   mem", 4);
  run(kstep<4, 1, 1, 1>, "K4 direct  prmt   mem", 4);
  run(kstep<4, 2, 0, 1>, "K4 mixed   isetp  mem", 4);
  run(kstep<4, 2, 1, 0>, "K4 mixed   prmt   reg", 4);
  run(kstep<4, 2, 1, 1>, "K4 mixed   prmt   mem", 4);
  return 0;
}
