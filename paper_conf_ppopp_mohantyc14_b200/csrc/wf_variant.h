// wf_variant.h -- the compiled kernel-variant table entry (host side, not part of the ABI).
#pragma once
#include <cstddef>
#include <cuda_runtime.h>

#include "wf_internal.h"

namespace wfk {

struct Variant {
  int fn, dsize, k, warps, skew;
  int threads;         // CTA size (compute warps + helper warps)
  size_t smem;
  const void* kernel;  // __global__ function pointer (for occupancy queries)
  cudaError_t (*launch)(const SweepLaunch&, cudaStream_t, size_t);
  int impl;            // kernel generation (SEQCMP: 4 = block hand-offs, 8 = lane pipeline)
  const void* alt[4];  // other instantiations launch() may pick for this variant (e.g. compile-time
                       // tsize); occupancy() takes the minimum over kernel and alt[]
  int strip;           // rows per hand-off block = rows per inter-slab message (generation 8: U);
                       // 0 = fixed by the generation (not selectable)
};

// SEQCMP v8 variants (wf_nw8.cu): global (dsize 0) and local / Smith-Waterman (dsize 1)
const Variant* nw8_table(size_t* n);
// SEQCMP local (Smith-Waterman) variants (wf_sw.cu); looked up with dsize = 1
const Variant* sw_table(size_t* n);
// SYNTHETIC v7 variants (wf_syn.cu)
const Variant* syn_table(size_t* n);

}  // namespace wfk
