// wf_sweep.cuh -- the persistent sm_100a band sweep.
//
// What it computes: a[i][j] = f(a[i-1][j], a[i][j-1], a[i-1][j-1], x_i, y_j) over the
// rows x cols interior (Sec. 1), for one column slab [c0, c1).
//
// How (B200-first; the paper's per-diagonal OpenCL launches, P:199-204 and Fig. 2, are
// prior art only):
//  * One launch per slab.  The slab is cut into column BANDS of band_w = WARPS*32*K
//    columns; a persistent CTA owns a band and sweeps all its rows, then takes band
//    b + gridDim.x.  All CTAs are co-resident (the host sizes the grid from occupancy).
//  * Inside a band, lane l of warp w owns K adjacent columns and keeps their previous
//    row (N and NW) in registers.  Lanes are skewed: at loop step t lane l is on row
//    t - D*l + 1, so the value it needs from its west neighbour (lane l-1's east
//    column) was produced D steps earlier and travels by __shfl_up_sync.  Cells on one
//    anti-diagonal of the band run in parallel across lanes -- the paper's observation
//    that "within a diagonal, computation of each data point is independent"
//     -- without any per-diagonal relaunch.
//  * Warp-to-warp and band-to-band west values travel as LL words (32-bit value +
//    32-bit tag in one 8-byte store, which is single-copy atomic), so a consumer
//    validates each row by its tag: no fences, no separate flags.  Within a CTA the
//    ring is in shared memory (tag = row); between bands/slabs it is a global ring
//    (tag = launch epoch), polled by a feeder warp and forwarded into shared memory.
//    The last slab band stores straight into the next slab's ring -- a peer (NVLink)
//    address when the next slab lives on another GPU.
//  * Each lane stages its K outputs in a per-warp shared-memory row ring; when a row
//    is complete in the warp (lane 31 passed it) the warp writes it out with
//    coalesced 16-byte stores: every output byte is written to HBM exactly once.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include "wf_internal.h"

namespace wfk {

constexpr int kHandSlots = 256;   // rows in each shared-memory handoff ring (power of 2)

__host__ __device__ constexpr int ring_rows(int D) {
  // rows alive in a warp's staging ring: lane 0 at row t+1, lane 31 at t-31D+1 -> 31D+1
  return (31 * D + 1) <= 32 ? 32 : (31 * D + 1) <= 64 ? 64 : (31 * D + 1) <= 128 ? 128 : 256;
}

__device__ __forceinline__ unsigned long long ld_relaxed_sys(const unsigned long long* p) {
  unsigned long long v;
  asm volatile("ld.relaxed.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_relaxed_sys(unsigned long long* p, unsigned long long v) {
  asm volatile("st.relaxed.sys.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ void st_relaxed_sys_u32(unsigned* p, unsigned v) {
  asm volatile("st.relaxed.sys.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ unsigned ld_relaxed_sys_u32(const unsigned* p) {
  unsigned v;
  asm volatile("ld.relaxed.sys.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
// GPU-scope LL accesses: band-to-band rings on one device need no system scope
__device__ __forceinline__ unsigned long long ld_relaxed_gpu(const unsigned long long* p) {
  unsigned long long v;
  asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_relaxed_gpu(unsigned long long* p, unsigned long long v) {
  asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ unsigned long long globaltimer() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
}
__device__ __forceinline__ unsigned long long lds_vol(const unsigned long long* p) {
  return *reinterpret_cast<const volatile unsigned long long*>(p);
}
__device__ __forceinline__ void sts_vol(unsigned long long* p, unsigned long long v) {
  *reinterpret_cast<volatile unsigned long long*>(p) = v;
}
__device__ __forceinline__ int lds_vol_i(const int* p) { return *reinterpret_cast<const volatile int*>(p); }
__device__ __forceinline__ void sts_vol_i(int* p, int v) { *reinterpret_cast<volatile int*>(p) = v; }
__device__ __forceinline__ unsigned long long ll_pack(uint32_t val, uint32_t tag) {
  return (static_cast<unsigned long long>(tag) << 32) | val;
}

// Race / liveness testing: a build with -DWF_JITTER=1 inserts pseudo-random
// back-offs (1 call in 8 sleeps up to ~1 us, warp-uniform) at the producers and consumers of
// every hand-off protocol, so parity under it checks the orderings for schedules the natural
// timing never produces.  A no-op in the product build.
#ifndef WF_JITTER
#define WF_JITTER 0
#endif
__device__ __forceinline__ void wf_jitter(unsigned salt) {
  if constexpr (WF_JITTER != 0) {
    unsigned h = static_cast<unsigned>(clock64() >> 4) ^ (salt * 0x9E3779B9u) ^ (blockIdx.x * 0x85EBCA6Bu) ^
                 ((threadIdx.x >> 5) * 0xC2B2AE35u);
    h = __shfl_sync(0xffffffffu, h, 0);   // one decision per warp
    h ^= h >> 16;
    h *= 0x7feb352du;
    h ^= h >> 15;
    if ((h & 7u) == 0) __nanosleep(h >> 22);
  }
}

// The device error word is epoch-tagged -- (epoch & 0x0FFFFFFF) << 4 | code -- so a
// failure of an earlier run never has to be cleared before the next launch.
__device__ __forceinline__ int err_word(const SweepLaunch& L, int code) {
  return static_cast<int>(((L.epoch & 0x0FFFFFFFu) << 4) | static_cast<unsigned>(code));
}
__device__ __forceinline__ bool run_failed(const SweepLaunch& L) {
  const int e = *reinterpret_cast<volatile int*>(L.err);
  return (static_cast<unsigned>(e) >> 4) == (L.epoch & 0x0FFFFFFFu) && (e & 15) != DEV_OK;
}

// Watchdog for dependency waits: returns true when the wait must be abandoned
// (budget exhausted -> sets the error word; or another CTA already failed).
struct Watchdog {
  long long t0;
  unsigned polls;
  __device__ __forceinline__ void start() { t0 = -1; polls = 0; }
  __device__ __forceinline__ bool expired(const SweepLaunch& L) {
    if ((++polls & 255u) != 0) return false;
    const long long now = clock64();
    if (t0 < 0) { t0 = now; return false; }
    if (run_failed(L)) return true;
    if (static_cast<unsigned long long>(now - t0) > L.watchdog) {
      atomicExch(L.err, err_word(L, DEV_TIMEOUT));
      return true;
    }
    return false;
  }
};

// Shared-memory carve-up for one CTA.
template <int NF, int K, int WARPS, int D>
struct Smem {
  static constexpr int kSlots = kHandSlots;
  static constexpr int R = ring_rows(D);
  static constexpr size_t stage_words = size_t(WARPS) * NF * R * 32 * K;     // u32
  static constexpr size_t hand_words = size_t(WARPS) * kHandSlots * NF;       // u64
  static constexpr size_t bytes = stage_words * 4 + hand_words * 8 + 16 * 4;
  uint32_t* stage;
  unsigned long long* hand;
  int* prog;
  __device__ __forceinline__ explicit Smem(unsigned char* base) {
    hand = reinterpret_cast<unsigned long long*>(base);
    stage = reinterpret_cast<uint32_t*>(base + hand_words * 8);
    prog = reinterpret_cast<int*>(base + hand_words * 8 + stage_words * 4);
  }
  __device__ __forceinline__ unsigned long long* hand_slot(int w, int row) const {
    return hand + (size_t(w) * kHandSlots + (row & (kHandSlots - 1))) * NF;
  }
  __device__ __forceinline__ uint32_t* stage_row(int w, int f, int row) const {
    return stage + ((size_t(w) * NF + f) * R + (row & (R - 1))) * (32 * K);
  }
};

// ---------------------------------------------------------------------------------
// Feeder warp: west input of the band's first column for every row, from the
// column-0 boundary (first band of slab 0) or from the band's global LL ring.
// ---------------------------------------------------------------------------------
template <class P, class SM>
__device__ __forceinline__ bool feeder(const SweepLaunch& L, const P& pol, const SM& sm, int band, int lane) {
  constexpr int NF = P::NF;
  const bool boundary = L.first_slab && band == 0;
  const unsigned long long* src = L.edge + size_t(band) * edge_stride(L.rows) * NF;   // slot r holds row r
  int base = 1, seen_prog = 0;
  Watchdog wd;
  wd.start();
  while (base <= L.rows) {
    wf_jitter(16);
    // back-pressure: rows base .. base+63 go to slots that held rows base-kSlots .. ;
    // those must have been consumed by compute warp 0.
    // The feeder is normally far ahead, so it sleeps between polls: a tight LDS spin would
    // occupy the SM's MIO pipe that the compute warps' SHFL/LDS/STS depend on.
    const int need = base + 63 - SM::kSlots;
    while (seen_prog < need) {
      seen_prog = lds_vol_i(sm.prog + 0);
      if (seen_prog < need) {
        if (wd.expired(L)) return false;
        __nanosleep(256);
      }
    }
    uint32_t v[2][NF];
    bool ok[2];
#pragma unroll
    for (int h = 0; h < 2; ++h) {
      const int r = base + h * 32 + lane;
      ok[h] = true;
      if (r <= L.rows) {
        if (boundary) {
          pol.left(r, v[h]);
        } else {
#pragma unroll
          for (int f = 0; f < NF; ++f) {
            const unsigned long long w = ld_relaxed_sys(src + size_t(r) * NF + f);
            v[h][f] = static_cast<uint32_t>(w);
            ok[h] = ok[h] && static_cast<uint32_t>(w >> 32) == L.epoch;
          }
        }
      }
    }
    const unsigned m0 = __ballot_sync(0xffffffffu, ok[0]);
    const unsigned m1 = __ballot_sync(0xffffffffu, ok[1]);
    int n = (m0 == 0xffffffffu) ? 32 + (__ffs(~m1) ? __ffs(~m1) - 1 : 32) : __ffs(~m0) - 1;
    if (base + n > L.rows + 1) n = L.rows + 1 - base;
#pragma unroll
    for (int h = 0; h < 2; ++h) {
      const int r = base + h * 32 + lane;
      if (r < base + n) {
        unsigned long long* slot = sm.hand_slot(0, r);
        // policies with a byte-sized row input (x_i of sequence comparison) ship it in the
        // tag's top byte, so compute warps never load it from global memory
        uint32_t tag = static_cast<uint32_t>(r);
        if constexpr (P::kTagRowIn) tag |= pol.row_in(r) << 24;
#pragma unroll
        for (int f = 0; f < NF; ++f) sts_vol(slot + f, ll_pack(v[h][f], tag));
      }
    }
    if (L.trace && lane == 0) {
      L.trace[size_t(band) * kTraceSlots + 40] += 1;
      if (n == 0) L.trace[size_t(band) * kTraceSlots + 41] += 1;
    }
    if (n == 0) {
      if (wd.expired(L)) return false;
      __nanosleep(128);
    } else if (n < 32) {
      __nanosleep(64);   // producer is just ahead: poll less often, let it run ahead
      wd.start();
    } else {
      wd.start();
    }
    base += n;
  }
  // the predecessor slab may now overwrite this band-0 ring in its next run
  if (!L.first_slab && band == 0 && L.ack_prev && lane == 0) st_relaxed_sys_u32(L.ack_prev, L.epoch);
  return true;
}

// ---------------------------------------------------------------------------------
// Compute warp: K columns per lane, rows swept with lane skew D.
// ---------------------------------------------------------------------------------
template <class P, int K, int WARPS, int D>
__device__ __forceinline__ bool compute_warp(const SweepLaunch& L, const P& pol, const Smem<P::NF, K, WARPS, D>& sm,
                                             int band, int warp, int lane) {
  constexpr int NF = P::NF;
  constexpr int R = Smem<NF, K, WARPS, D>::R;
  const int rows = L.rows;
  const int jb = L.c0 + band * L.band_w + (warp * 32 + lane) * K;   // 0-based global column of lane's 1st column
  // per-column inputs and the boundary row 0
  uint32_t cin[K];
  uint32_t Np[K][NF];
  uint32_t prevW[NF];
#pragma unroll
  for (int m = 0; m < K; ++m) {
    const int j1 = jb + m + 1;                  // 1-based column
    const bool vc = (jb + m) < L.c1;
    cin[m] = vc ? pol.col_in(j1) : 0u;
    pol.top(vc ? j1 : 0, Np[m]);
  }
  pol.top(jb < L.c1 ? jb : 0, prevW);           // H[0][jb] (jb is the 1-based west column)

  uint32_t q[D][NF];
#pragma unroll
  for (int d = 0; d < D; ++d)
#pragma unroll
    for (int f = 0; f < NF; ++f) q[d][f] = 0u;

  const bool lane_has_cols = jb < L.c1;
  const bool lane_full = jb + K <= L.c1;
  const int64_t pitch = L.pitch;
  const int jrel = jb - L.c0;                   // column offset inside the slab's planes

  int seen_prog_next = 0;                       // producer view of warp+1's consumption
  uint32_t xr_next = 0;
  {
    const int r0 = 1 - D * lane;
    if (r0 >= 1 && r0 <= rows) xr_next = pol.row_in(r0);
  }
  Watchdog wd;
  const int T = rows + 31 * D;
  const int trace_every = (rows + kTraceRows - 1) / kTraceRows;
  for (int t = 0; t < T; ++t) {
    const int row = t - D * lane + 1;
    const bool active = row >= 1 && row <= rows;
    if (L.trace && warp == 0 && lane == 0 && t < rows && (t % trace_every) == 0)
      L.trace[size_t(band) * kTraceSlots + t / trace_every] = globaltimer();
    const uint32_t xr = xr_next;
    {
      const int rn = row + 1;
      xr_next = (rn >= 1 && rn <= rows) ? pol.row_in(rn) : 0u;
    }
    // ---- west input: lane 0 from the handoff ring (row t+1), others from lane-1 via q
    uint32_t Win[NF];
#pragma unroll
    for (int f = 0; f < NF; ++f) Win[f] = q[D - 1][f];
    if (t < rows) {
      const int r = t + 1;
      const unsigned long long* slot = sm.hand_slot(warp, r);
      uint32_t got[NF];
      wf_jitter(17);
      wd.start();
      for (;;) {
        bool ok = true;
#pragma unroll
        for (int f = 0; f < NF; ++f) {
          const unsigned long long w = lds_vol(slot + f);
          got[f] = static_cast<uint32_t>(w);
          ok = ok && static_cast<uint32_t>(w >> 32) == static_cast<uint32_t>(r);
        }
        if (ok) break;
        if (wd.expired(L)) return false;
      }
      if (lane == 0) {
#pragma unroll
        for (int f = 0; f < NF; ++f) Win[f] = got[f];
        sts_vol_i(sm.prog + warp, r);           // row r consumed: its slot may be reused
      }
    }
    // ---- the cells of this lane's row segment
    if (active) {
      uint32_t H[K][NF];
#pragma unroll
      for (int m = 0; m < K; ++m) {
        const uint32_t* NWm = (m == 0) ? prevW : Np[m - 1];
        const uint32_t* Wm = (m == 0) ? Win : H[m - 1];
        pol.cell(Np[m], Wm, NWm, xr, cin[m], H[m]);
      }
#pragma unroll
      for (int f = 0; f < NF; ++f) {
        prevW[f] = Win[f];
#pragma unroll
        for (int m = 0; m < K; ++m) Np[m][f] = H[m][f];
      }
      // stage the K outputs of each plane in the warp's row ring
#pragma unroll
      for (int f = 0; f < NF; ++f) {
        uint32_t* dst = sm.stage_row(warp, f, row) + lane * K;
        if constexpr (K == 4) {
          *reinterpret_cast<uint4*>(dst) = make_uint4(H[0][f], H[1][f], H[2][f], H[3][f]);
        } else if constexpr (K == 2) {
          *reinterpret_cast<uint2*>(dst) = make_uint2(H[0][f], H[1][f]);
        } else if constexpr (K == 8) {
          reinterpret_cast<uint4*>(dst)[0] = make_uint4(H[0][f], H[1][f], H[2][f], H[3][f]);
          reinterpret_cast<uint4*>(dst)[1] = make_uint4(H[4][f], H[5][f], H[6][f], H[7][f]);
        } else {
#pragma unroll
          for (int m = 0; m < K; ++m) dst[m] = H[m][f];
        }
      }
    }
    // ---- pass the east column to the next lane (value for its row D steps later)
#pragma unroll
    for (int f = 0; f < NF; ++f) {
      const uint32_t r = __shfl_up_sync(0xffffffffu, Np[K - 1][f], 1);
#pragma unroll
      for (int d = D - 1; d > 0; --d) q[d][f] = q[d - 1][f];
      q[0][f] = r;
    }
    // ---- lane 31 publishes its east column (row t-31D+1) to the next warp / band / slab
    const int r31 = t - 31 * D + 1;
    if (r31 >= 1 && r31 <= rows) {
      if (warp < WARPS - 1) {
        const int need = r31 - kHandSlots;      // slot's previous row must be consumed
        if (seen_prog_next < need) {
          wd.start();
          for (;;) {
            seen_prog_next = lds_vol_i(sm.prog + warp + 1);
            if (seen_prog_next >= need) break;
            if (wd.expired(L)) return false;
          }
        }
        if (lane == 31) {
          unsigned long long* slot = sm.hand_slot(warp + 1, r31);
#pragma unroll
          for (int f = 0; f < NF; ++f) sts_vol(slot + f, ll_pack(Np[K - 1][f], static_cast<uint32_t>(r31)));
        }
      } else {
        const bool to_next_slab = band + 1 >= L.nbands;
        if (to_next_slab && r31 == 1 && L.next_edge && L.ack_self) {
          // the next slab must have drained this ring in the previous run (warp-uniform wait)
          wd.start();
          for (;;) {
            const unsigned a = ld_relaxed_sys_u32(L.ack_self);
            if (static_cast<int>(a - (L.epoch - 1u)) >= 0) break;
            if (wd.expired(L)) return false;
          }
        }
        unsigned long long* dst = to_next_slab ? L.next_edge : L.edge + size_t(band + 1) * edge_stride(rows) * NF;
        if (dst && lane == 31) {
#pragma unroll
          for (int f = 0; f < NF; ++f) st_relaxed_sys(dst + size_t(r31) * NF + f, ll_pack(Np[K - 1][f], L.epoch));
        }
      }
    }
    __syncwarp();
    // ---- write out the row that just completed in this warp
    if (r31 >= 1 && r31 <= rows && lane_has_cols) {
#pragma unroll
      for (int f = 0; f < NF; ++f) {
        const uint32_t* src = sm.stage_row(warp, f, r31) + lane * K;
        uint32_t* dst = static_cast<uint32_t*>(L.out[f]) + int64_t(r31 - 1) * pitch + jrel;
        if (lane_full) {
          if constexpr (K == 4) {
            *reinterpret_cast<uint4*>(dst) = *reinterpret_cast<const uint4*>(src);
          } else if constexpr (K == 2) {
            *reinterpret_cast<uint2*>(dst) = *reinterpret_cast<const uint2*>(src);
          } else if constexpr (K == 8) {
            reinterpret_cast<uint4*>(dst)[0] = reinterpret_cast<const uint4*>(src)[0];
            reinterpret_cast<uint4*>(dst)[1] = reinterpret_cast<const uint4*>(src)[1];
          } else {
#pragma unroll
            for (int m = 0; m < K; ++m) dst[m] = src[m];
          }
        } else {
#pragma unroll
          for (int m = 0; m < K; ++m)
            if (jb + m < L.c1) dst[m] = src[m];
        }
      }
    }
    __syncwarp();
  }
  if (L.trace && warp == 0 && lane == 0) L.trace[size_t(band) * kTraceSlots + kTraceRows] = globaltimer();
  (void)R;
  return true;
}

template <class P, int K, int WARPS, int D>
__global__ void __launch_bounds__((WARPS + 1) * 32) sweep_kernel(const SweepLaunch L, const P pol) {
  using S = Smem<P::NF, K, WARPS, D>;
  extern __shared__ __align__(16) unsigned char smem_raw[];
  const S sm(smem_raw);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  for (int band = blockIdx.x; band < L.nbands; band += gridDim.x) {
    for (int i = threadIdx.x; i < WARPS * kHandSlots * P::NF; i += blockDim.x) sm.hand[i] = 0ull;
    if (threadIdx.x < WARPS) sm.prog[threadIdx.x] = 0;
    __syncthreads();
    bool ok;
    if (warp == WARPS) ok = feeder(L, pol, sm, band, lane);
    else ok = compute_warp<P, K, WARPS, D>(L, pol, sm, band, warp, lane);
    (void)ok;
    __syncthreads();
    if (run_failed(L)) return;
  }
}

}  // namespace wfk
