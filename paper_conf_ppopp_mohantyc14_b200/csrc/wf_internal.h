// wf_internal.h -- host-side launch interface between the C-ABI layer (wf_api.cpp)
// and the sm_100a kernels (wf_sweep.cu).  Not part of the public ABI.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include "../../include/wf.h"

namespace wfk {

// Everything one slab's persistent launch needs.
struct SweepLaunch {
  // problem
  int32_t fn, rows, cols, tsize, dsize;
  int32_t c0, c1;                 // slab interior columns [c0, c1), 0-based (the output planes' columns)
  int32_t cc0;                    // first computed column: c0 - halo (NEXT-4 overlap bands), else c0
  int32_t halo_bands;             // leading overlap bands (outputs to halo_out), 0 without a halo
  int32_t export_band;            // the band whose east edge goes to next_edge (nbands-1 without a halo)
  void* halo_out;                 // overlap bands' scratch plane: rows x halo_pitch int32
  int64_t halo_pitch;
  int32_t match, mismatch, gap;
  int32_t alphabet;               // SEQCMP: 0 = any byte codes, 1..8 = codes < alphabet
  // tuning
  int32_t k, warps, skew;         // lane columns, compute warps per CTA, lane skew
  int32_t band_w, nbands;         // band_w = warps*32*k
  int32_t grid;                   // persistent CTAs (all co-resident)
  // io
  const void* row_in;
  const void* col_in;
  const void* top[WF_MAX_PLANES];
  const void* left[WF_MAX_PLANES];
  void* out[WF_MAX_PLANES];
  int64_t pitch;
  // edges: edge[b] (b = 0..nbands-1) is band b's inbound LL ring, rows*nf u64 each.
  // edge[0] of slab g > 0 is written by slab g-1 (possibly through a peer mapping).
  unsigned long long* edge;
  unsigned long long* next_edge;  // inbound ring of slab g+1's band 0 (NULL on the last slab)
  // Cross-run back-pressure between slabs: slab g+1's band-0 feeder stores the epoch it has
  // fully consumed into slab g's ack word (ack_prev, possibly a peer address); slab g waits
  // for ack_self >= epoch-1 before its first store into next_edge.
  unsigned* ack_self;
  unsigned* ack_prev;
  int32_t first_slab;             // 1: band 0's west input is the column-0 boundary
  uint32_t epoch;
  int* err;                       // device error word
  // Optional timeline (WF_TRACE=1): per band kTraceSlots globaltimer stamps written by
  // compute warp 0 lane 0 every rows/kTraceRows rows, plus feeder poll counters.
  unsigned long long* trace;
  unsigned long long watchdog;
  // SEQCMP local = 1 (Smith-Waterman): per lane (best value, first row reaching it),
  // [nbands][warps][32]; the slab's best cell (value, 1-based row, 1-based global column)
  int32_t local;
  int32_t cluster;
  int32_t impl;        // wf_params.kernel actually used (0 = the function's default generation)
  int32_t strip;       // wf_params.strip: rows per hand-off block (generation 8); 0 = the default
  int2* lane_best;
  int32_t* best_out;
};

// LL slots per band ring and cell word: slot r holds row r (1..rows); padded to an even
// count so every band's ring starts 16-byte aligned (vector LL stores).
__host__ __device__ inline size_t edge_stride(int rows) { return size_t((rows + 2) & ~1); }

// Words per cell (= output planes) for a function.
int nwords(int fn, int dsize);
// Dynamic shared memory the kernel variant needs; <0 if the variant is not compiled.
int smem_bytes(const SweepLaunch& L);
// Max co-resident CTAs per SM for the variant (0 if it cannot launch).
int occupancy(const SweepLaunch& L, int smem);
// Launch (asynchronous).  Returns cudaSuccess or the launch error.
cudaError_t launch(const SweepLaunch& L, cudaStream_t s);
// Finish the Smith-Waterman best-cell reduction of a run (after the sweep, same stream).
cudaError_t launch_sw_best(const SweepLaunch& L, cudaStream_t s);
// Is (fn, dsize, k, warps, skew) compiled?  (SEQCMP: dsize carries the local flag.)
bool variant_exists(int fn, int dsize, int k, int warps, int skew, int impl = 0, int strip = 0);
// Rows per hand-off block of the variant that runs (generation 8: its U; 0 for the others).
int variant_strip(int fn, int dsize, int k, int warps, int skew, int impl, int strip);

constexpr int kTraceSlots = 64;   // per band: [0..32] row stamps, [40] feeder polls, [41] empty polls,
constexpr int kTraceRows = 32;    // [42] last warp's first outbound stamp

// Error word codes (device side).
enum : int { DEV_OK = 0, DEV_TIMEOUT = 1 };

}  // namespace wfk
