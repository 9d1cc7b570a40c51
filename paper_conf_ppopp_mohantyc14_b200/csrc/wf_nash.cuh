// wf_nash.cuh -- the Nash-equilibrium stand-in sweep (
// DESIGN.md reading R8): every cell solves one n x n bimatrix game whose payoffs are
// derived from a key hashed over (N, NW, x_i, y_j, W), and emits four words
//   p0 = number of pure Nash equilibria, p1 = first one (row-major index, -1 if none),
//   p2 = A at p1 (-1), p3 = B at p1 (-1).
//
// Design (B200-first; a cell is ~n^2 hashes + two max-reductions, far too much work for
// one lane): ONE WARP PER COLUMN.  A CTA owns a band of WARPS adjacent columns; warp w
// sweeps all rows of column band*WARPS + w, and the 32 lanes cooperate on each cell:
//  * the W-independent part of the key chain (N, NW, x_i, y_j) is hashed before waiting
//    for the west value, so only four hashes sit on the column-to-column critical path;
//  * the n^2 payoff pairs are generated 32 at a time (lane l owns entries l, l+32, ...),
//    parked in a per-warp shared-memory scratch as bytes;
//  * column maxima of A and row maxima of B are one task per lane (2n tasks);
//  * equilibrium flags are combined with __ballot_sync: popc gives p0, the lowest set
//    bit of the first non-empty ballot gives p1 (entries are visited in row-major order).
// West values travel exactly as in the generic band sweep (wf_sweep.cuh): four LL words
// per row through a shared-memory ring between the warps of a CTA, through the band's
// global LL ring between CTAs / slabs (fed by the feeder warp).
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include "wf_sweep.cuh"

namespace wfk {

constexpr uint32_t kNashSeed = 0x9E3779B9u;   // DESIGN.md R8 (same constant as the oracle's definition)
constexpr int kNashMaxN = 64;

__device__ __forceinline__ uint32_t lowbias32(uint32_t x) {
  x ^= x >> 16;
  x *= 0x7feb352du;
  x ^= x >> 15;
  x *= 0x846ca68bu;
  x ^= x >> 16;
  return x;
}

struct PolNash {
  static constexpr int NF = 4;
  static constexpr bool kTagRowIn = false;
  const uint32_t* r;            // x_i: rows entries
  const uint32_t* c;            // y_j: cols entries
  const int32_t* topp[4];       // boundary row 0, cols+1 entries per plane (index = 1-based column)
  const int32_t* leftp[4];      // boundary column 0, rows+1 entries per plane (index 0 unused)
  __device__ __forceinline__ uint32_t row_in(int i) const { return __ldg(r + (i - 1)); }
  __device__ __forceinline__ uint32_t col_in(int j) const { return __ldg(c + (j - 1)); }
  __device__ __forceinline__ void top(int j, uint32_t* w) const {
#pragma unroll
    for (int p = 0; p < 4; ++p) w[p] = static_cast<uint32_t>(__ldg(topp[p] + j));
  }
  __device__ __forceinline__ void left(int i, uint32_t* w) const {
#pragma unroll
    for (int p = 0; p < 4; ++p) w[p] = static_cast<uint32_t>(__ldg(leftp[p] + i));
  }
};

// Shared memory: inbound LL rings (one per warp), consumption counters, and per-warp
// game scratch (A, B as bytes, column maxima of A, row maxima of B).
#ifndef WF_NASH_REDUX_ROWMAX
#define WF_NASH_REDUX_ROWMAX 0   // 1: row maxima of B by half-warp REDUX instead of a shuffle butterfly
#endif

template <int WARPS>
struct NashSmem {
  static constexpr int kSlots = 128;                                        // rows per ring
  static constexpr size_t hand_words = size_t(WARPS) * kSlots * 4;           // u64
  static constexpr size_t fixed_bytes = hand_words * 8 + 16 * 4;
  static size_t scratch_bytes(int n) { return (size_t(2) * n * n + 2 * n + 15) & ~size_t(15); }
  __host__ static size_t bytes(int n) { return fixed_bytes + WARPS * scratch_bytes(n); }
  unsigned long long* hand;
  int* prog;
  uint8_t* scratch;
  int scratch_stride;
  __device__ __forceinline__ NashSmem(unsigned char* base, int n) {
    hand = reinterpret_cast<unsigned long long*>(base);
    prog = reinterpret_cast<int*>(base + hand_words * 8);
    scratch = base + fixed_bytes;
    scratch_stride = static_cast<int>((2 * n * n + 2 * n + 15) & ~15);
  }
  __device__ __forceinline__ unsigned long long* hand_slot(int w, int row) const {
    return hand + (size_t(w) * kSlots + (row & (kSlots - 1))) * 4;
  }
};

// Rest of lowbias32 after its first xorshift (x is already x0 ^ (x0 >> 16)), masked to the
// payoff byte.
__device__ __forceinline__ uint32_t lowbias32_tail_byte(uint32_t x) {
  x *= 0x7feb352du;
  x ^= x >> 15;
  x *= 0x846ca68bu;
  return (x ^ (x >> 16)) & 255u;
}

// n = 16 fast path: the 256 entries stay in registers.  Lane l owns column b = l & 15 and
// rows a = (l >> 4) + 2k, k = 0..7, i.e. entries idx = l + 32k (row-major order, so ballot k
// covers entries 32k .. 32k+31).  Payoff hash of entry idx: lowbias32(key ^ c), c = 2 idx
// (A) or 2 idx + 1 (B); c < 2^16 so the first xorshift folds: x1 = (key ^ key >> 16) ^ c.
__device__ __forceinline__ void nash_solve16(uint32_t key, int lane, uint32_t o[4]) {
  const uint32_t KL = (key ^ (key >> 16)) ^ (2u * static_cast<uint32_t>(lane));
  uint32_t A[8], B[8];
#pragma unroll
  for (int k = 0; k < 8; ++k) {
    const uint32_t x = KL ^ (64u * k);
    A[k] = lowbias32_tail_byte(x);
    B[k] = lowbias32_tail_byte(x ^ 1u);
  }
  // column maxima of A: over the lane's 8 rows, then with the partner half (l ^ 16)
  uint32_t cA = A[0];
#pragma unroll
  for (int k = 1; k < 8; ++k) cA = max(cA, A[k]);
  cA = max(cA, __shfl_xor_sync(0xffffffffu, cA, 16));
  // row maxima of B: row (l >> 4) + 2k spans the 16 lanes of the half -> butterfly over
  // xor 1, 2, 4, 8 on two rows at a time (16-bit SIMD max)
  uint32_t P[4];
#if WF_NASH_REDUX_ROWMAX
  // each half-warp is one group of the reduction (row (l >> 4) + 2k lives in one half)
  const unsigned half = (lane < 16) ? 0x0000FFFFu : 0xFFFF0000u;
#pragma unroll
  for (int q = 0; q < 4; ++q)
    P[q] = __reduce_max_sync(half, B[2 * q]) | (__reduce_max_sync(half, B[2 * q + 1]) << 16);
#else
#pragma unroll
  for (int q = 0; q < 4; ++q) P[q] = B[2 * q] | (B[2 * q + 1] << 16);
#pragma unroll
  for (int s = 1; s < 16; s <<= 1) {
#pragma unroll
    for (int q = 0; q < 4; ++q) P[q] = __vmaxu2(P[q], __shfl_xor_sync(0xffffffffu, P[q], s));
  }
#endif
  // pure equilibria of the lane's 8 entries as a bit mask, then two warp reductions (REDUX):
  // the count, and the smallest row-major index 32k + lane holding one (the first
  // equilibrium); its payoffs come from the lane that owns it (one shuffle each)
  uint32_t mask = 0, kmin = 8, selA = 0, selB = 0;
#pragma unroll
  for (int k = 7; k >= 0; --k) {   // descending: the selects end on the smallest k
    const uint32_t rB = (k & 1) ? (P[k >> 1] >> 16) : (P[k >> 1] & 0xFFFFu);
    const bool ne = A[k] == cA && B[k] == rB;
    mask |= ne ? (1u << k) : 0u;
    kmin = ne ? static_cast<uint32_t>(k) : kmin;
    selA = ne ? A[k] : selA;
    selB = ne ? B[k] : selB;
  }
  const int count = static_cast<int>(__reduce_add_sync(0xffffffffu, static_cast<unsigned>(__popc(mask))));
  const uint32_t mine = mask ? 32u * kmin + static_cast<uint32_t>(lane) : 0xFFFFFFFFu;
  const uint32_t firstu = __reduce_min_sync(0xffffffffu, mine);
  const int first = firstu == 0xFFFFFFFFu ? -1 : static_cast<int>(firstu);
  const int src = first < 0 ? 0 : (first & 31);
  uint32_t pa = __shfl_sync(0xffffffffu, selA, src);
  uint32_t pb = __shfl_sync(0xffffffffu, selB, src);
  if (first < 0) pa = pb = 0xFFFFFFFFu;
  o[0] = static_cast<uint32_t>(count);
  o[1] = static_cast<uint32_t>(first);
  o[2] = pa;
  o[3] = pb;
}

// Any n (1..64): payoffs parked as bytes in the warp's shared scratch; entries visited 32 at
// a time in row-major order (lane l owns entries l, l + 32, ...).
__device__ __forceinline__ void nash_solve_smem(uint32_t key, int lane, int n, uint8_t* scratch, uint32_t o[4]) {
  const int nn = n * n;
  const int rounds = (nn + 31) >> 5;
  uint8_t* sA = scratch;
  uint8_t* sB = sA + nn;
  uint8_t* sCol = sB + nn;
  uint8_t* sRow = sCol + n;
  for (int k = 0, idx = lane; k < rounds; ++k, idx += 32) {
    if (idx < nn) {
      sA[idx] = static_cast<uint8_t>(lowbias32(key ^ (2u * idx)) & 255u);
      sB[idx] = static_cast<uint8_t>(lowbias32(key ^ (2u * idx + 1u)) & 255u);
    }
  }
  __syncwarp();
  // best responses: column maxima of A (tasks 0..n-1), row maxima of B (tasks n..2n-1)
  for (int t = lane; t < 2 * n; t += 32) {
    uint32_t m = 0;
    if (t < n) {
      for (int a = 0; a < n; ++a) m = max(m, static_cast<uint32_t>(sA[a * n + t]));
      sCol[t] = static_cast<uint8_t>(m);
    } else {
      const uint8_t* row = sB + (t - n) * n;
      for (int b = 0; b < n; ++b) m = max(m, static_cast<uint32_t>(row[b]));
      sRow[t - n] = static_cast<uint8_t>(m);
    }
  }
  __syncwarp();
  // lane's first entry (a, b) and the per-round step (+32 entries)
  int a = lane / n, b = lane - (lane / n) * n;
  const int da = 32 / n, db = 32 - da * n;
  int count = 0, first = -1;
  for (int k = 0, idx = lane; k < rounds; ++k, idx += 32) {
    const bool ne = idx < nn && sA[idx] == sCol[b] && sB[idx] == sRow[a];
    const unsigned bal = __ballot_sync(0xffffffffu, ne);
    count += __popc(bal);
    if (first < 0 && bal) first = 32 * k + __ffs(bal) - 1;
    a += da;
    b += db;
    if (b >= n) { b -= n; ++a; }
  }
  o[0] = static_cast<uint32_t>(count);
  o[1] = static_cast<uint32_t>(first);
  o[2] = first >= 0 ? static_cast<uint32_t>(sA[first]) : 0xFFFFFFFFu;
  o[3] = first >= 0 ? static_cast<uint32_t>(sB[first]) : 0xFFFFFFFFu;
  __syncwarp();   // scratch is rewritten by the next cell
}

template <int WARPS, int NS>
__device__ __forceinline__ bool nash_warp(const SweepLaunch& L, const PolNash& pol, const NashSmem<WARPS>& sm,
                                          int band, int warp, int lane) {
  const int j = L.c0 + band * WARPS + warp;                 // 0-based global column
  if (j >= L.c1) return true;                               // past the slab (ragged last band)
  const int rows = L.rows;
  const int64_t pitch = L.pitch;
  const int jrel = j - L.c0;
  const bool east_local = warp < WARPS - 1;
  const bool east_exists = east_local ? (j + 1 < L.c1) : true;

  const uint32_t cj = pol.col_in(j + 1);
  uint32_t N[4], NW[4];
  pol.top(j + 1, N);
  pol.top(j, NW);
  uint32_t xr_next = pol.row_in(1);
  int seen_prog_next = 0;
  // per-lane loop invariants (kept out of the row loop: no parameter-space reloads)
  // output: lane p < 4 writes plane p of this column
  uint32_t* const out_lane = static_cast<uint32_t*>(lane == 0 ? L.out[0] : lane == 1 ? L.out[1] : lane == 2 ? L.out[2] : L.out[3]) + jrel;
  const bool writer = lane < 4;
  // east handoff: lane p < 4 stores word p of the LL row into the next warp's shared ring
  // (tag = row) or into the next band's / slab's global ring (tag = epoch)
  unsigned long long* const east_smem = (east_local && east_exists) ? sm.hand + size_t(warp + 1) * NashSmem<WARPS>::kSlots * 4 + lane : nullptr;
  unsigned long long* east_glob = nullptr;
  if (!east_local) {
    const bool to_next_slab = band + 1 >= L.nbands;
    unsigned long long* g = to_next_slab ? L.next_edge : L.edge + size_t(band + 1) * edge_stride(rows) * 4;
    east_glob = g ? g + lane : nullptr;
  }
  const bool wait_ack = !east_local && east_glob && band + 1 >= L.nbands && L.ack_self;
  const uint32_t epoch = L.epoch;
  const unsigned long long* const in_ring = sm.hand + size_t(warp) * NashSmem<WARPS>::kSlots * 4;
  const bool tracer = L.trace && warp == 0 && lane == 0;
  Watchdog wd;
#ifdef WF_NASH_PROF
  long long ph[4] = {0, 0, 0, 0};
  long long tp = clock64();
#define NASH_PH(i) do { const long long _n = clock64(); ph[i] += _n - tp; tp = _n; } while (0)
#else
#define NASH_PH(i) do { } while (0)
#endif
  const int trace_every = (rows + kTraceRows - 1) / kTraceRows;
  int trace_next = 0;   // next traced row index (0-based)
  int64_t out_off = 0;
  for (int r = 1; r <= rows; ++r) {
    const uint32_t xr = xr_next;
    if (r < rows) xr_next = pol.row_in(r + 1);
    // W-independent prefix of the key chain: N.p0..3, NW.p0..3, x_i, y_j
    uint32_t key = kNashSeed;
#pragma unroll
    for (int p = 0; p < 4; ++p) key = lowbias32(key ^ N[p]);
#pragma unroll
    for (int p = 0; p < 4; ++p) key = lowbias32(key ^ NW[p]);
    key = lowbias32(key ^ xr);
    key = lowbias32(key ^ cj);
    NASH_PH(0);
    // west value of row r
    uint32_t W[4];
    {
      const unsigned long long* slot = in_ring + (r & (NashSmem<WARPS>::kSlots - 1)) * 4;
      wf_jitter(18);
      wd.start();
      for (;;) {
        bool ok = true;
#pragma unroll
        for (int p = 0; p < 4; ++p) {
          const unsigned long long w = lds_vol(slot + p);
          W[p] = static_cast<uint32_t>(w);
          ok = ok && static_cast<uint32_t>(w >> 32) == static_cast<uint32_t>(r);
        }
        if (ok) break;
        if (wd.expired(L)) return false;
        // a waiting warp must not steal issue slots from the computing ones: back off for
        // the minimum sleep quantum (~80 cycles, profiles/r01_microbench.txt mb7)
        __nanosleep(16);
      }
      // consumption is reported every 32 rows (the producer's window is kSlots = 128 rows)
      if ((r & 31) == 0 || r == rows) {
        __syncwarp();
        if (lane == 0) sts_vol_i(sm.prog + warp, r);
      }
    }
    // timeline (WF_TRACE=1): when warp 0 received the west value of every (rows/32)-th row
    if (tracer && r - 1 == trace_next) {
      L.trace[size_t(band) * kTraceSlots + (r - 1) / trace_every] = globaltimer();
      trace_next += trace_every;
    }
    NASH_PH(1);
#pragma unroll
    for (int p = 0; p < 4; ++p) key = lowbias32(key ^ W[p]);

    uint32_t o[4];
    if constexpr (NS == 16) {
      nash_solve16(key, lane, o);
    } else {
      nash_solve_smem(key, lane, L.tsize, sm.scratch + size_t(warp) * sm.scratch_stride, o);
    }
    NASH_PH(2);

    // output planes and the east handoff (selects, not o[lane]: o stays in registers)
    const uint32_t mine = lane == 0 ? o[0] : lane == 1 ? o[1] : lane == 2 ? o[2] : o[3];
    if (writer) out_lane[out_off] = mine;
    out_off += pitch;
    if (east_smem) {
      const int need = r - NashSmem<WARPS>::kSlots;
      if (seen_prog_next < need) {
        wd.start();
        for (;;) {
          seen_prog_next = lds_vol_i(sm.prog + warp + 1);
          if (seen_prog_next >= need) break;
          if (wd.expired(L)) return false;
          __nanosleep(16);
        }
      }
      if (writer) sts_vol(east_smem + (r & (NashSmem<WARPS>::kSlots - 1)) * 4, ll_pack(mine, static_cast<uint32_t>(r)));
    } else if (east_glob) {
      if (r == 1 && wait_ack) {
        // the next slab must have drained this ring in the previous run
        wd.start();
        for (;;) {
          const unsigned a = ld_relaxed_sys_u32(L.ack_self);
          if (static_cast<int>(a - (epoch - 1u)) >= 0) break;
          if (wd.expired(L)) return false;
        }
      }
      if (writer) st_relaxed_sys(east_glob + size_t(r) * 4, ll_pack(mine, epoch));
    }
#pragma unroll
    for (int p = 0; p < 4; ++p) {
      NW[p] = W[p];
      N[p] = o[p];
    }
    NASH_PH(3);
  }
#ifdef WF_NASH_PROF
  if (tracer)
    for (int i = 0; i < 4; ++i) L.trace[size_t(band) * kTraceSlots + 48 + i] = ph[i];
#endif
#undef NASH_PH
  if (L.trace && lane == 0) {
    if (warp == 0) L.trace[size_t(band) * kTraceSlots + kTraceRows] = globaltimer();
    if (warp == WARPS - 1) L.trace[size_t(band) * kTraceSlots + 42] = globaltimer();
  }
  return true;
}

template <int WARPS, int NS>
__global__ void __launch_bounds__((WARPS + 1) * 32, WARPS >= 8 ? 4 : 8) nash_kernel(const SweepLaunch L, const PolNash pol) {
  extern __shared__ __align__(16) unsigned char nash_smem_raw[];
  const NashSmem<WARPS> sm(nash_smem_raw, L.tsize);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  for (int band = blockIdx.x; band < L.nbands; band += gridDim.x) {
    for (int i = threadIdx.x; i < int(NashSmem<WARPS>::hand_words); i += blockDim.x) sm.hand[i] = 0ull;
    if (threadIdx.x < WARPS) sm.prog[threadIdx.x] = 0;
    __syncthreads();
    if (warp == WARPS) feeder(L, pol, sm, band, lane);
    else nash_warp<WARPS, NS>(L, pol, sm, band, warp, lane);
    __syncthreads();
    if (run_failed(L)) return;
  }
}

}  // namespace wfk
