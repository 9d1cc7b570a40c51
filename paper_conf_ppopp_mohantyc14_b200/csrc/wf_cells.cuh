// wf_cells.cuh -- cell functions f(N, W, NW, x_i, y_j) of the paper's applications,
// as device policies for the band sweep (wf_sweep.cuh).  Each policy states the cell as a
// sequence of single IEEE/integer operations in a FIXED order with W entering last
// (readings R5, R11), so results are bit-identical to any sequential evaluation.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

namespace wfk {

// --- Sequence comparison: Needleman-Wunsch, linear gap (
//     BASELINE.json "Needleman-Wunsch integer scores"; reading R9/R10).
//     H = max(max(NW + s, N + g), W + g): two DPX VIADDMNMX, W last.
struct PolSeq {
  static constexpr int NF = 1;
  static constexpr bool kTagRowIn = true;   // x_i travels in the LL tag's top byte
  const uint8_t* x;
  const uint8_t* y;
  int32_t match, mismatch, gap;
  __device__ __forceinline__ uint32_t row_in(int i) const { return __ldg(x + (i - 1)); }
  __device__ __forceinline__ uint32_t col_in(int j) const { return __ldg(y + (j - 1)); }
  __device__ __forceinline__ void top(int j, uint32_t* w) const { w[0] = static_cast<uint32_t>(j * gap); }
  __device__ __forceinline__ void left(int i, uint32_t* w) const { w[0] = static_cast<uint32_t>(i * gap); }
  __device__ __forceinline__ void cell(const uint32_t* N, const uint32_t* W, const uint32_t* NW, uint32_t xi,
                                       uint32_t yj, uint32_t* o) const {
    const int s = (xi == yj) ? match : mismatch;
    const int t = __viaddmax_s32(static_cast<int>(N[0]), gap, static_cast<int>(NW[0]) + s);
    o[0] = static_cast<uint32_t>(__viaddmax_s32(static_cast<int>(W[0]), gap, t));
  }
};

// --- Synthetic application (Sec. 3.1.1; readings R4-R6).
//     Words: 0 = i0, 1 = i1, 2.. = f[d] (fp32 bits).  Explicit _rn intrinsics: no FMA
//     contraction, no reassociation (nvcc would otherwise contract a*b+c).
template <int DS>
struct PolSyn {
  static constexpr int NF = 2 + DS;
  static constexpr bool kTagRowIn = false;
  const float* u;
  const float* v;
  const float* topf[DS > 0 ? DS : 1];
  const float* leftf[DS > 0 ? DS : 1];
  int32_t tsize;
  __device__ __forceinline__ uint32_t row_in(int i) const {
    if constexpr (DS > 0) return __float_as_uint(__ldg(u + (i - 1)));
    else return 0u;
  }
  __device__ __forceinline__ uint32_t col_in(int j) const {
    if constexpr (DS > 0) return __float_as_uint(__ldg(v + (j - 1)));
    else return 0u;
  }
  __device__ __forceinline__ void top(int j, uint32_t* w) const {
    w[0] = static_cast<uint32_t>(-1);
    w[1] = 0u;
#pragma unroll
    for (int d = 0; d < DS; ++d) w[2 + d] = __float_as_uint(__ldg(topf[d] + j));
  }
  __device__ __forceinline__ void left(int i, uint32_t* w) const {
    w[0] = static_cast<uint32_t>(-1);
    w[1] = 0u;
#pragma unroll
    for (int d = 0; d < DS; ++d) w[2 + d] = __float_as_uint(__ldg(leftf[d] + i));
  }
  __device__ __forceinline__ void cell(const uint32_t* N, const uint32_t* W, const uint32_t* NW, uint32_t ui,
                                       uint32_t vj, uint32_t* o) const {
    o[0] = static_cast<uint32_t>(max(max(static_cast<int>(N[0]), static_cast<int>(NW[0])), static_cast<int>(W[0])) + 1);
    o[1] = ((N[1] - NW[1]) + 1u) + W[1];
    if constexpr (DS > 0) {
      const float THIRD = __uint_as_float(0x3EAAAAABu);   // fp32 nearest 1/3
      const float A = __uint_as_float(0x3F7FF000u);       // 1 - 2^-12
      const float SCALE = __uint_as_float(0x39800000u);   // 2^-12
      const float c = __fmul_rn(__fmul_rn(__uint_as_float(ui), __uint_as_float(vj)), SCALE);
      float x[DS];
#pragma unroll
      for (int d = 0; d < DS; ++d)
        x[d] = __fmul_rn(__fadd_rn(__fadd_rn(__uint_as_float(N[2 + d]), __uint_as_float(NW[2 + d])),
                                   __uint_as_float(W[2 + d])),
                         THIRD);
      for (int t = 0; t < tsize; ++t) {
#pragma unroll
        for (int d = 0; d < DS; ++d) x[d] = __fmaf_rn(x[d], A, c);
      }
#pragma unroll
      for (int d = 0; d < DS; ++d) o[2 + d] = __float_as_uint(x[d]);
    }
  }
};

}  // namespace wfk
