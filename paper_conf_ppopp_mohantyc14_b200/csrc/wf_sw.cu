// wf_sw.cu -- Smith-Waterman local alignment ("Smith-Waterman", P:432-435;
// SURVEY.md §8(f) NEXT-1; R9): the v4 sequence-comparison sweep (wf_nw.cuh) with
// LOCAL = true -- H = max(0, NW + s, N + g, W + g), boundary 0 -- plus the best-cell
// reduction: every lane tracks its best value and the first row reaching it inside the sweep;
// sw_best_kernel turns those into the slab's first (row-major) best cell.
#include <cstring>

#include <cuda.h>
#include <cudaTypedefs.h>

#include "wf_cells.cuh"
#include "wf_nw.cuh"
#include "wf_sweep.cuh"
#include "wf_variant.h"

namespace wfk {

cudaError_t encode_plane_map(CUtensorMap* m, const SweepLaunch& L, int box_cols, int box_rows);
cudaError_t launch_nw_kernel(void (*kfn)(const SweepLaunch, const PolSeq, const CUtensorMap), const SweepLaunch& L,
                             const PolSeq& pol, const CUtensorMap& tmap, int threads, size_t smem, cudaStream_t s);

// One CTA: value max, then the smallest row among the lanes holding it, then the smallest
// column of that row whose cell holds it (read back from the output plane).
__global__ void __launch_bounds__(1024) sw_best_kernel(const int2* __restrict__ lb, int n, const int32_t* __restrict__ H,
                                                      int64_t pitch, int width, int c0, int k, int band_w, int warps,
                                                      int32_t* out) {
  __shared__ int s_best, s_row, s_col;
  if (threadIdx.x == 0) {
    s_best = 0;
    s_row = 0x7fffffff;
    s_col = 0x7fffffff;
  }
  __syncthreads();
  int b = 0;
  for (int i = threadIdx.x; i < n; i += blockDim.x) b = max(b, lb[i].x);
  atomicMax(&s_best, b);
  __syncthreads();
  const int vb = s_best;
  for (int i = threadIdx.x; i < n; i += blockDim.x)
    if (vb > 0 && lb[i].x == vb) atomicMin(&s_row, lb[i].y);
  __syncthreads();
  const int rb = s_row;
  for (int i = threadIdx.x; i < n; i += blockDim.x) {
    if (vb > 0 && lb[i].x == vb && lb[i].y == rb) {
      const int band = i / (warps * 32), warp = (i / 32) % warps, lane = i % 32;
      const int j0 = band * band_w + warp * 32 * k + lane * k;
      for (int m = 0; m < k; ++m)
        if (j0 + m < width && H[int64_t(rb - 1) * pitch + j0 + m] == vb) {
          atomicMin(&s_col, j0 + m);
          break;
        }
    }
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    // every cell is >= 0: with no positive cell the first best cell is (1, first column)
    out[0] = vb;
    out[1] = vb > 0 ? rb : 1;
    out[2] = c0 + (vb > 0 ? s_col : 0) + 1;
  }
}

cudaError_t launch_sw_best(const SweepLaunch& L, cudaStream_t s) {
  const int n = L.nbands * L.warps * 32;
  sw_best_kernel<<<1, 1024, 0, s>>>(L.lane_best, n, static_cast<const int32_t*>(L.out[0]), L.pitch, L.c1 - L.c0, L.c0,
                                    L.k, L.band_w, L.warps, L.best_out);
  return cudaGetLastError();
}

namespace {

template <int K, int W, int D, int U>
cudaError_t launch_sw(const SweepLaunch& L, cudaStream_t s, size_t smem) {
  PolSeq pol{};
  pol.x = static_cast<const uint8_t*>(L.row_in);
  pol.y = static_cast<const uint8_t*>(L.col_in);
  pol.match = L.match;
  pol.mismatch = L.mismatch;
  pol.gap = L.gap;
  CUtensorMap tmap;
  cudaError_t e = encode_plane_map(&tmap, L, 32 * K, U);
  if (e != cudaSuccess) return e;
  auto kfn = (L.alphabet >= 1 && L.alphabet <= 8) ? nw_kernel<K, W, D, U, true, true> : nw_kernel<K, W, D, U, false, true>;
  e = cudaFuncSetAttribute(kfn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  return launch_nw_kernel(kfn, L, pol, tmap, (W + 2) * 32, smem, s);
}

template <int K, int W, int D>
Variant make_sw() {
  constexpr int U = K >= 8 ? 16 : 32;
  using S = NwSmem<K, W, D, U>;
  // dsize = 1 marks the local (Smith-Waterman) variant of SEQCMP in the variant table
  return Variant{WF_FN_SEQCMP, 1, K, W, D, (W + 2) * 32, S::bytes,
                 reinterpret_cast<const void*>(nw_kernel<K, W, D, U, true, true>), &launch_sw<K, W, D, U>, 4,
                 {reinterpret_cast<const void*>(nw_kernel<K, W, D, U, false, true>)}};
}

}  // namespace

const Variant* sw_table(size_t* n) {
#ifdef WF_MIN_VARIANTS
  static const Variant v[] = {make_sw<4, 2, 1>()};
#else
  static const Variant v[] = {make_sw<4, 2, 1>(), make_sw<4, 1, 1>(), make_sw<2, 2, 1>(), make_sw<2, 4, 1>(),
                              make_sw<8, 1, 1>(), make_sw<4, 1, 2>(), make_sw<2, 2, 2>(), make_sw<1, 2, 1>()};
#endif
  *n = sizeof(v) / sizeof(v[0]);
  return v;
}

}  // namespace wfk
