// wf_sweep.cu -- instantiations and host-side launch of the persistent band sweep.
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <type_traits>

#include <cuda.h>
#include <cudaTypedefs.h>

#include "wf_cells.cuh"
#include "wf_nash.cuh"
#include "wf_nw.cuh"
#include "wf_sweep.cuh"
#include "wf_variant.h"

namespace wfk {

int nwords(int fn, int dsize) {
  switch (fn) {
    case WF_FN_SEQCMP: return 1;
    case WF_FN_SYNTHETIC: return 2 + dsize;
    case WF_FN_NASH: return 4;
    default: return 0;
  }
}

namespace {

template <class P, int K, int W, int D>
cudaError_t launch_t(const SweepLaunch& L, cudaStream_t s, size_t smem) {
  P pol{};
  if constexpr (std::is_same<P, PolSeq>::value) {
    pol.x = static_cast<const uint8_t*>(L.row_in);
    pol.y = static_cast<const uint8_t*>(L.col_in);
    pol.match = L.match;
    pol.mismatch = L.mismatch;
    pol.gap = L.gap;
  } else {
    pol.u = static_cast<const float*>(L.row_in);
    pol.v = static_cast<const float*>(L.col_in);
    for (int d = 0; d < L.dsize && d < (int)(sizeof(pol.topf) / sizeof(pol.topf[0])); ++d) {
      pol.topf[d] = static_cast<const float*>(L.top[d]);
      pol.leftf[d] = static_cast<const float*>(L.left[d]);
    }
    pol.tsize = L.tsize;
  }
  auto kfn = sweep_kernel<P, K, W, D>;
  cudaError_t e = cudaFuncSetAttribute(kfn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  kfn<<<L.grid, (W + 1) * 32, smem, s>>>(L, pol);
  return cudaGetLastError();
}

template <class P, int K, int W, int D>
Variant make_variant(int fn, int dsize) {
  using S = Smem<P::NF, K, W, D>;
  return Variant{fn, dsize, K, W, D, (W + 1) * 32, S::bytes, reinterpret_cast<const void*>(sweep_kernel<P, K, W, D>),
                 &launch_t<P, K, W, D>, 4};
}

}  // namespace

// cuTensorMapEncodeTiled through the runtime's driver entry point (no -lcuda link needed)
cudaError_t encode_plane_map_f(CUtensorMap* m, const SweepLaunch& L, int plane, int box_cols, int box_rows) {
  static PFN_cuTensorMapEncodeTiled_v12000 enc = nullptr;
  if (!enc) {
    void* fp = nullptr;
    cudaDriverEntryPointQueryResult q;
    cudaError_t e = cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fp, cudaEnableDefault, &q);
    if (e != cudaSuccess || q != cudaDriverEntryPointSuccess || !fp) return cudaErrorNotSupported;
    enc = reinterpret_cast<PFN_cuTensorMapEncodeTiled_v12000>(fp);
  }
  const cuuint64_t dims[2] = {static_cast<cuuint64_t>(L.c1 - L.c0), static_cast<cuuint64_t>(L.rows)};
  const cuuint64_t strides[1] = {static_cast<cuuint64_t>(L.pitch) * 4};
  const cuuint32_t box[2] = {static_cast<cuuint32_t>(box_cols), static_cast<cuuint32_t>(box_rows)};
  const cuuint32_t estr[2] = {1, 1};
  CUresult r = enc(m, CU_TENSOR_MAP_DATA_TYPE_INT32, 2, L.out[plane], dims, strides, box, estr,
                   CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_NONE,
                   CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  return r == CUDA_SUCCESS ? cudaSuccess : cudaErrorInvalidValue;
}
// int32 [rows][cols] plane at `base` with a row pitch of pitch_elems elements
cudaError_t encode_map_2d(CUtensorMap* m, void* base, int cols, int rows, int64_t pitch_elems, int box_cols, int box_rows) {
  SweepLaunch L{};
  L.c0 = 0;
  L.c1 = cols;
  L.rows = rows;
  L.pitch = pitch_elems;
  L.out[0] = base;
  return encode_plane_map_f(m, L, 0, box_cols, box_rows);
}
cudaError_t encode_plane_map(CUtensorMap* m, const SweepLaunch& L, int box_cols, int box_rows) {
  return encode_plane_map_f(m, L, 0, box_cols, box_rows);
}

namespace {

}  // namespace

// Launch an NW-family kernel of generation 4 as a plain persistent grid.
cudaError_t launch_nw_kernel(void (*kfn)(const SweepLaunch, const PolSeq, const CUtensorMap), const SweepLaunch& L,
                             const PolSeq& pol, const CUtensorMap& tmap, int threads, size_t smem, cudaStream_t s) {
  SweepLaunch Lp = L;
  Lp.cluster = 0;
  kfn<<<L.grid, threads, smem, s>>>(Lp, pol, tmap);
  return cudaGetLastError();
}

namespace {

template <int K, int W, int D, int U>
cudaError_t launch_nw(const SweepLaunch& L, cudaStream_t s, size_t smem) {
  PolSeq pol{};
  pol.x = static_cast<const uint8_t*>(L.row_in);
  pol.y = static_cast<const uint8_t*>(L.col_in);
  pol.match = L.match;
  pol.mismatch = L.mismatch;
  pol.gap = L.gap;
  // TMA descriptor of this slab's output plane: int32 [rows][slab cols], row pitch in bytes,
  // box = one warp's 32*K columns x U rows (the steady-state write-out unit)
  CUtensorMap tmap;
  cudaError_t e = encode_plane_map(&tmap, L, 32 * K, U);
  if (e != cudaSuccess) return e;
  // alphabet 1..8 promises codes < 8: byte-permute score lookup; otherwise compare+select
  auto kfn = (L.alphabet >= 1 && L.alphabet <= 8) ? nw_kernel<K, W, D, U, true> : nw_kernel<K, W, D, U, false>;
  e = cudaFuncSetAttribute(kfn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  return launch_nw_kernel(kfn, L, pol, tmap, (W + 2) * 32, smem, s);   // + I/O warp + x-staging warp
}

template <int K, int W, int D>
Variant make_nw_variant() {
#ifndef WF_NW_U
#define WF_NW_U 32
#endif
  constexpr int U = K >= 8 ? 16 : WF_NW_U;   // rows per block (TMA box height)
  using S = NwSmem<K, W, D, U>;
  return Variant{WF_FN_SEQCMP, 0, K, W, D, (W + 2) * 32, S::bytes,
                 reinterpret_cast<const void*>(nw_kernel<K, W, D, U, true>),
                 &launch_nw<K, W, D, U>, 4, {reinterpret_cast<const void*>(nw_kernel<K, W, D, U, false>)}};
}

template <int W>
cudaError_t launch_nash(const SweepLaunch& L, cudaStream_t s, size_t smem) {
  PolNash pol{};
  pol.r = static_cast<const uint32_t*>(L.row_in);
  pol.c = static_cast<const uint32_t*>(L.col_in);
  for (int p = 0; p < 4; ++p) {
    pol.topp[p] = static_cast<const int32_t*>(L.top[p]);
    pol.leftp[p] = static_cast<const int32_t*>(L.left[p]);
  }
  auto kfn = L.tsize == 16 ? nash_kernel<W, 16> : nash_kernel<W, 0>;   // n = 16: register fast path
  cudaError_t e = cudaFuncSetAttribute(kfn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  kfn<<<L.grid, (W + 1) * 32, smem, s>>>(L, pol);
  return cudaGetLastError();
}

// NASH: one warp per column (lane_cols = 1, skew = 1); smem listed without the per-warp
// game scratch, which depends on n (added by smem_bytes()).
template <int W>
Variant make_nash_variant() {
  return Variant{WF_FN_NASH, 0, 1, W, 1, (W + 1) * 32, NashSmem<W>::fixed_bytes,
                 reinterpret_cast<const void*>(nash_kernel<W, 16>), &launch_nash<W>, 4,
                 {reinterpret_cast<const void*>(nash_kernel<W, 0>)}};
}

// --- the compiled variant set -------------------------------------------------------
#define WF_SEQ(K, W, D) make_nw_variant<K, W, D>()
#define WF_SYN(DS, K, W, D) make_variant<PolSyn<DS>, K, W, D>(WF_FN_SYNTHETIC, DS)
#define WF_NASH(W) make_nash_variant<W>()
#define WF_SYN_DS(DS) WF_SYN(DS, 1, 1, 1), WF_SYN(DS, 1, 2, 1), WF_SYN(DS, 1, 4, 1), WF_SYN(DS, 2, 1, 1), \
    WF_SYN(DS, 2, 2, 1), WF_SYN(DS, 1, 2, 2), WF_SYN(DS, 2, 2, 2)

const Variant* table(size_t* n) {
#ifdef WF_MIN_VARIANTS   // quick experimental builds (tools/ablate.sh)
  static const Variant v[] = {WF_SEQ(4, 1, 1), WF_SEQ(4, 1, 2), WF_SEQ(4, 2, 1), WF_SEQ(4, 3, 1), WF_SEQ(2, 1, 1), WF_SEQ(8, 1, 1),
                              WF_NASH(8), WF_NASH(2)};
#else
  static const Variant v[] = {
      WF_SEQ(2, 1, 1), WF_SEQ(2, 2, 1), WF_SEQ(2, 4, 1), WF_SEQ(2, 1, 2), WF_SEQ(2, 2, 2), WF_SEQ(2, 4, 2),
      WF_SEQ(2, 2, 3), WF_SEQ(2, 4, 3),
      WF_SEQ(4, 1, 1), WF_SEQ(4, 2, 1), WF_SEQ(4, 3, 1), WF_SEQ(4, 4, 1), WF_SEQ(4, 1, 2), WF_SEQ(4, 2, 2), WF_SEQ(4, 4, 2),
      WF_SEQ(4, 1, 3), WF_SEQ(4, 2, 3),
      WF_SEQ(8, 1, 1), WF_SEQ(8, 2, 1), WF_SEQ(8, 1, 2), WF_SEQ(8, 2, 2),
      WF_SEQ(1, 1, 1), WF_SEQ(1, 2, 1), WF_SEQ(1, 4, 1),
      WF_SYN_DS(0), WF_SYN_DS(1), WF_SYN_DS(2), WF_SYN_DS(3), WF_SYN_DS(4),
      WF_SYN_DS(5), WF_SYN_DS(6), WF_SYN_DS(7), WF_SYN_DS(8),
      WF_NASH(1), WF_NASH(2), WF_NASH(4), WF_NASH(8),
  };
#endif
  *n = sizeof(v) / sizeof(v[0]);
  return v;
}

const Variant* find(int fn, int dsize, int k, int warps, int skew, int impl, int strip) {
  size_t n;
  // SEQCMP: generation 8 (the default, wf_nw8.cu) for its compiled (K, warps, strip) at skew 1;
  // every other tuning -- or kernel = 4 -- runs generation 4 (wf_nw.cuh, wf_sw.cu).  strip 0 =
  // generation 8's default block (the first entry of a (K, warps) in its table).
  if (fn == WF_FN_SEQCMP && skew == 1 && (impl == 0 || impl == 8)) {
    const Variant* t8 = nw8_table(&n);
    for (size_t i = 0; i < n; ++i)
      if (t8[i].dsize == dsize && t8[i].k == k && t8[i].warps == warps && (strip == 0 || t8[i].strip == strip))
        return &t8[i];
    if (impl == 8 || strip != 0) return nullptr;
  }
  if (strip != 0) return nullptr;   // the other generations' blocks are fixed
  if (fn == WF_FN_SEQCMP && dsize == 1) {   // local alignment (Smith-Waterman)
    const Variant* ts = sw_table(&n);
    for (size_t i = 0; i < n; ++i)
      if (ts[i].k == k && ts[i].warps == warps && ts[i].skew == skew) return &ts[i];
    return nullptr;
  }
  if (fn == WF_FN_SYNTHETIC && impl == 8) {   // plane-split wf_syn only; no fallback
    const Variant* t7 = syn_table(&n);
    for (size_t i = 0; i < n; ++i)
      if (t7[i].impl == 8 && t7[i].dsize == dsize && t7[i].k == k && t7[i].warps == warps && t7[i].skew == skew)
        return &t7[i];
    return nullptr;
  }
  if (fn == WF_FN_SYNTHETIC && skew == 1 && impl != 4) {   // wf_syn unless generation 4 (the generic sweep) is asked
    const Variant* t7 = syn_table(&n);
    for (size_t i = 0; i < n; ++i)   // a wf_syn variant whose staging rings do not fit falls back to the generic sweep
      if (t7[i].impl == 7 && t7[i].dsize == dsize && t7[i].k == k && t7[i].warps == warps && t7[i].smem <= 232448)
        return &t7[i];
  }
  const Variant* t = table(&n);
  for (size_t i = 0; i < n; ++i)
    if (t[i].fn == fn && t[i].dsize == dsize && t[i].k == k && t[i].warps == warps && t[i].skew == skew) return &t[i];
  return nullptr;
}

}  // namespace

bool variant_exists(int fn, int dsize, int k, int warps, int skew, int impl, int strip) {
  // compiled AND within the 227 KB per-CTA shared-memory limit of sm_100
  const Variant* v = find(fn, (fn == WF_FN_SYNTHETIC || fn == WF_FN_SEQCMP) ? dsize : 0, k, warps, skew, impl, strip);
  return v != nullptr && v->smem <= 232448;
}

int variant_strip(int fn, int dsize, int k, int warps, int skew, int impl, int strip) {
  const Variant* v = find(fn, (fn == WF_FN_SYNTHETIC || fn == WF_FN_SEQCMP) ? dsize : 0, k, warps, skew, impl, strip);
  return v ? v->strip : 0;
}

int smem_bytes(const SweepLaunch& L) {
  const Variant* v = find(L.fn, L.fn == WF_FN_SYNTHETIC ? L.dsize : (L.fn == WF_FN_SEQCMP ? L.local : 0), L.k, L.warps, L.skew, L.impl, L.strip);
  if (!v) return -1;
  if (L.fn == WF_FN_NASH) return (int)(v->smem + size_t(L.warps) * ((size_t(2) * L.tsize * L.tsize + 2 * L.tsize + 15) & ~size_t(15)));
  return (int)v->smem;
}

int occupancy(const SweepLaunch& L, int smem) {
  const Variant* v = find(L.fn, L.fn == WF_FN_SYNTHETIC ? L.dsize : (L.fn == WF_FN_SEQCMP ? L.local : 0), L.k, L.warps, L.skew, L.impl, L.strip);
  if (!v) return 0;
  if (cudaFuncSetAttribute(v->kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, smem) != cudaSuccess) {
    cudaGetLastError();
    return 0;
  }
  // every instantiation launch() may pick must be co-resident at the grid size (all CTAs spin
  // on each other): the minimum over the variant's kernel and its alternatives
  int best = -1;
  for (int i = -1; i < 4; ++i) {
    const void* k = i < 0 ? v->kernel : v->alt[i];
    if (!k) continue;
    if (cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, smem) != cudaSuccess) {
      cudaGetLastError();
      return 0;
    }
    int blocks = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&blocks, k, v->threads, smem) != cudaSuccess) {
      cudaGetLastError();
      return 0;
    }
    best = best < 0 ? blocks : (blocks < best ? blocks : best);
  }
  return best < 0 ? 0 : best;
}

cudaError_t launch(const SweepLaunch& L, cudaStream_t s) {
  const Variant* v = find(L.fn, L.fn == WF_FN_SYNTHETIC ? L.dsize : (L.fn == WF_FN_SEQCMP ? L.local : 0), L.k, L.warps, L.skew, L.impl, L.strip);
  if (!v) return cudaErrorInvalidDeviceFunction;
  return v->launch(L, s, (size_t)smem_bytes(L));
}

int variant_count() {
  size_t n;
  table(&n);
  return (int)n;
}

}  // namespace wfk
