// wf_nw7.cu -- sequence-comparison (Needleman-Wunsch / PAPER.md P:432-435) band sweep,
// version 7: per-row west hand-offs.
//
// Same band / lane model as wf_nw.cuh (v4): a persistent CTA owns a band of WARPS*32*K
// columns and sweeps all its rows; lane l of a warp owns K adjacent columns and at step t
// is on row t - l + 1, so the west input of every lane but lane 0 is its left neighbour's
// east value of the previous step -- the paper's "within a diagonal, computation of each
// data point is independent" without per-diagonal launches.  What v7 changes,
// because the v4 phase profile (profiles/r01_microbench.txt) showed the band-to-band hop
// (~186 rows, 127 hops = 40 % of C4) and not the cell was the loss:
//
//  * West inputs of a warp are 8-byte LL words in a shared ring, ONE PER ROW:
//        bits 0..31 west value, 32..47 row selector (score byte-permute selector, or the
//        raw residue code), 48..63 tag = row & 0xffff.
//    Warp w > 0's ring is written by lane 31 of warp w-1 (one STS.64 per step); warp 0's
//    by the I/O warp (from the column-0 boundary, or the band's global LL ring that lane
//    31 of the previous band's last warp stores into -- one st.relaxed.sys per row, a peer
//    NVLink address for the slab edge).  A consumer waits on its own rows only: no block
//    published progress counters, no fences (the tag validates each 8-byte word).
//  * Rotation: lane 31's east value has no right neighbour inside the warp, so its slot in
//    the per-step lane rotation carries lane 0's NEXT west word (preloaded for a block of
//    U rows by vector loads that every lane issues, broadcast): one shuffle for the value
//    and one for the selector per step; the row code travels with the value, no x ring.
//  * Outputs: per-warp staging ring (row-major, 32K int32 per row) -> one TMA 2-D tensor
//    store per U-row block (UTMASTG), as in v4; every output byte is written once.
//  * Cell, W entering last (R9):  t1 = max(N + g, NW + s);  H = max(W + g, t1)
//    (two VIADDMNMX), or the prefix form of v4 (FORM = 1).
#include <cstdio>
#include <cstdlib>
#include <cstring>

#include <cuda.h>
#include <cudaTypedefs.h>

#include "wf_cells.cuh"
#include "wf_nw.cuh"
#include "wf_sweep.cuh"
#include "wf_variant.h"

namespace wfk {

constexpr int kLL7 = 256;
#ifndef WF_NW7_PUB
#define WF_NW7_PUB 0   // write-back: 1 = coalesced 16-B stores from the staging ring per block, 0 = TMA 2-D store per 2 blocks
#endif
#ifndef WF_NW7_ABL
#define WF_NW7_ABL 0   // performance archaeology only (wrong grids): 1 no publish, 2 no west-tag waits, 4 no staging STS
#endif   // rows per west LL ring (power of 2, multiple of U)

__device__ __forceinline__ void lds_v2_u64(const unsigned long long* p, unsigned long long& a, unsigned long long& b) {
  asm volatile("ld.volatile.shared.v2.u64 {%0, %1}, [%2];"
               : "=l"(a), "=l"(b)
               : "r"(static_cast<uint32_t>(__cvta_generic_to_shared(p))));
}
__device__ __forceinline__ void sts_u64(unsigned long long* p, unsigned long long v) {
  asm volatile("st.volatile.shared.u64 [%0], %1;" ::"r"(static_cast<uint32_t>(__cvta_generic_to_shared(p))), "l"(v));
}
// predicated (branch-free) stores: a divergent `if (lane == 31)` around them would make the
// compiler wrap every following shuffle in a reconvergence sequence
__device__ __forceinline__ void sts_u64_if(bool p, unsigned long long* a, unsigned long long v) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q st.volatile.shared.u64 [%0], %1; }" ::"r"(
                   static_cast<uint32_t>(__cvta_generic_to_shared(a))),
               "l"(v), "r"(static_cast<int>(p))
               : "memory");
}
__device__ __forceinline__ void stg_sys_u64_if(bool p, unsigned long long* a, unsigned long long v) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q st.relaxed.sys.global.u64 [%0], %1; }" ::"l"(a), "l"(v),
               "r"(static_cast<int>(p))
               : "memory");
}
__device__ __forceinline__ unsigned long long ll7(int32_t v, uint32_t sel, int row) {
  return (static_cast<unsigned long long>((static_cast<uint32_t>(row) << 16) | (sel & 0xffffu)) << 32) |
         static_cast<uint32_t>(v);
}
__device__ __forceinline__ int ll7_slot(int row) { return (row - 2) & (kLL7 - 1); }

template <int K, int WARPS, int U>
struct Nw7Smem {
  // staging rows alive: lane skew (31) + this block (U) + the TMA group of two blocks in
  // flight + the group before it being released -> 4U + 31 <= R
  static constexpr int R = WF_NW7_PUB ? ((2 * U + 31) <= 64 ? 64 : 128) : ((4 * U + 31) <= 64 ? 64 : (4 * U + 31) <= 128 ? 128 : 256);
  static constexpr int ROWB = 32 * K * 4;
  static constexpr size_t stage_bytes = size_t(WARPS) * R * ROWB;
  static constexpr size_t ll_bytes = size_t(WARPS + 1) * kLL7 * 8;
  static constexpr size_t bytes = 1024 + stage_bytes + ll_bytes + 64 * 4;
  unsigned char* stage;     // [WARPS][R][32K] int32, 1024-byte aligned (TMA source)
  unsigned long long* ll;   // [WARPS+1][kLL7]: ring w = west input of warp w; ring WARPS = band east edge
  int* rprog;               // rprog[w]: rows of ring w consumed by its reader
  __device__ __forceinline__ explicit Nw7Smem(unsigned char* raw) {
    const uint32_t a = static_cast<uint32_t>(__cvta_generic_to_shared(raw));
    unsigned char* base = raw + ((1024u - (a & 1023u)) & 1023u);
    stage = base;
    ll = reinterpret_cast<unsigned long long*>(base + stage_bytes);
    rprog = reinterpret_cast<int*>(base + stage_bytes + ll_bytes);
  }
};

template <int K, int WARPS, int U, bool PRMT, int FORM>
struct Nw7Warp {
  using S = Nw7Smem<K, WARPS, U>;
  static constexpr int R = S::R;
  static constexpr int ROWB = S::ROWB;
  static_assert(U == 8 || U == 16, "block height");
  static_assert(kLL7 % U == 0 && R % (2 * U) == 0 && 32 % U == 0, "alignment");
  // staging slot of row r is (r + kOff) & (R-1): lane 31's rows of two blocks (t0-U-30 ..
  // t0-30+U-1, t0 an odd multiple of U) then occupy contiguous slots -- one TMA box
  static constexpr int kOff = 30 % (2 * U);

  const SweepLaunch& L;
  const CUtensorMap* tmap;
  const S& sm;
  const int band, warp, lane;
  int rows;
  int32_t gap, mmatch, mmis;
  int32_t gk[K];
  uint32_t qlo[K], qhi[K];
  uint32_t ycode[K];
  int32_t Np[K];             // N of the current row (the lane's previous row)
  int32_t prevW;             // NW of the current row's first column
  int32_t t1[K];             // max(N + g, NW + s) of the current row (FORM 0), or its prefix max (FORM 1)
  int wcol;
  unsigned char* stage_lane;
  uint32_t stage_w_s;
  const unsigned long long* myll;
  unsigned long long* nextll;  // next warp's ring, or the band's east-edge ring (last warp)
  Watchdog wd;

  __device__ __forceinline__ Nw7Warp(const SweepLaunch& L_, const CUtensorMap* tmap_, const S& sm_, int band_, int warp_,
                                     int lane_)
      : L(L_), tmap(tmap_), sm(sm_), band(band_), warp(warp_), lane(lane_) {
    rows = L.rows;
    gap = L.gap;
    mmatch = L.match;
    mmis = L.mismatch;
#pragma unroll
    for (int m = 0; m < K; ++m) gk[m] = (m + 1) * gap;
    const uint8_t* y = static_cast<const uint8_t*>(L.col_in);
    wcol = band * L.band_w + warp * 32 * K;
    const int jb = L.c0 + wcol + lane * K;
#pragma unroll
    for (int m = 0; m < K; ++m) {
      const bool vc = jb + m < L.c1;
      const uint32_t yc = vc ? static_cast<uint32_t>(__ldg(y + jb + m)) : 0xFFu;
      ycode[m] = yc;
      uint32_t lo = 0, hi = 0;
#pragma unroll
      for (int c = 0; c < 4; ++c) {
        lo |= (static_cast<uint32_t>(c == static_cast<int>(yc) ? mmatch : mmis) & 0xFFu) << (8 * c);
        hi |= (static_cast<uint32_t>(c + 4 == static_cast<int>(yc) ? mmatch : mmis) & 0xFFu) << (8 * c);
      }
      qlo[m] = lo;
      qhi[m] = hi;
      Np[m] = vc ? (jb + m + 1) * gap : 0;   // H[0][j] = j*g
    }
    prevW = jb < L.c1 ? jb * gap : 0;        // H[0][jb]
    unsigned char* stage_w = sm.stage + size_t(warp) * R * ROWB;
    stage_lane = stage_w + lane * (4 * K);
    stage_w_s = static_cast<uint32_t>(__cvta_generic_to_shared(stage_w));
    myll = sm.ll + size_t(warp) * kLL7;
    nextll = sm.ll + size_t(warp + 1) * kLL7;
  }

  __device__ __forceinline__ int32_t score(uint32_t sel, int m) const {
    if constexpr (PRMT) return prmt_s8(qlo[m], qhi[m], sel);
    else return (sel == ycode[m]) ? mmatch : mmis;
  }

  // The W-independent part of the next row's cells (off the lane-to-lane chain): needs only
  // the lane's own previous row (Np, prevW) and the row's selector.
  __device__ __forceinline__ void prep(uint32_t sel) {
#pragma unroll
    for (int m = 0; m < K; ++m) {
      const int32_t NW = m == 0 ? prevW : Np[m - 1];
      t1[m] = __viaddmax_s32(Np[m], gap, NW + score(sel, m));
      if constexpr (FORM == 1) {
        if (m > 0) t1[m] = __viaddmax_s32(t1[m - 1], gap, t1[m]);   // prefix max P_m
      }
    }
  }

  // W enters last: H_m = max(H_{m-1} + g, t1_m) (FORM 0) or max(W + (m+1)g, P_m) (FORM 1)
  __device__ __forceinline__ void cells(int32_t Win, int32_t (&H)[K]) const {
#pragma unroll
    for (int m = 0; m < K; ++m) {
      if constexpr (FORM == 1) H[m] = __viaddmax_s32(Win, gk[m], t1[m]);
      else H[m] = __viaddmax_s32(m == 0 ? Win : H[m - 1], gap, t1[m]);
    }
  }

  __device__ __forceinline__ void stage_store(int row, const int32_t (&H)[K]) const {
    if constexpr ((WF_NW7_ABL & 4) != 0) {
      if (row != -12345) return;
    }
    unsigned char* dst = stage_lane + ((row + kOff) & (R - 1)) * ROWB;
    if constexpr (K == 4) {
      *reinterpret_cast<int4*>(dst) = make_int4(H[0], H[1], H[2], H[3]);
    } else if constexpr (K == 2) {
      *reinterpret_cast<int2*>(dst) = make_int2(H[0], H[1]);
    } else if constexpr (K == 8) {
      reinterpret_cast<int4*>(dst)[0] = make_int4(H[0], H[1], H[2], H[3]);
      reinterpret_cast<int4*>(dst)[1] = make_int4(H[4], H[5], H[6], H[7]);
    } else {
#pragma unroll
      for (int m = 0; m < K; ++m) reinterpret_cast<int32_t*>(dst)[m] = H[m];
    }
  }

  __device__ __forceinline__ void write_row(int r) const {
    const int jrel = wcol + lane * K;
    const int width = L.c1 - L.c0;
    const uint32_t* src = reinterpret_cast<const uint32_t*>(stage_lane + ((r + kOff) & (R - 1)) * ROWB);
    uint32_t* dst = static_cast<uint32_t*>(L.out[0]) + int64_t(r - 1) * L.pitch + jrel;
    if (jrel + K <= width) {
      if constexpr (K == 4) {
        *reinterpret_cast<uint4*>(dst) = *reinterpret_cast<const uint4*>(src);
        return;
      } else if constexpr (K == 2) {
        *reinterpret_cast<uint2*>(dst) = *reinterpret_cast<const uint2*>(src);
        return;
      } else if constexpr (K == 8) {
        reinterpret_cast<uint4*>(dst)[0] = reinterpret_cast<const uint4*>(src)[0];
        reinterpret_cast<uint4*>(dst)[1] = reinterpret_cast<const uint4*>(src)[1];
        return;
      }
    }
#pragma unroll
    for (int m = 0; m < K; ++m)
      if (jrel + m < width) dst[m] = src[m];
  }

  // Load the U west words of rows r0 .. r0+U-1 (slots contiguous: r0 - 2 is a multiple of U)
  // until every word with row <= rows carries its row tag.  Every lane loads (broadcast).
  // The tag test is a tree of integer ORs: a `ok = ok && ...` chain compiles to a serial
  // chain of predicated compares (~16 dependent predicate ops, ~400 cycles per block).
  // Issue the loads of the U west words of rows r0 .. r0+U-1 (slots contiguous: r0 - 2 is a
  // multiple of U).  Every lane loads (broadcast).  ps keeps the raw high word: selector in
  // bits 0..15 (PRMT reads only those), tag (row & 0xffff) in bits 16..31.
  __device__ __forceinline__ void issue_block(int r0, uint32_t (&pv)[U], uint32_t (&ps)[U]) const {
    const unsigned long long* p = myll + ll7_slot(r0);
#pragma unroll
    for (int u = 0; u < U; u += 2) {
      unsigned long long a, b;
      lds_v2_u64(p + u, a, b);
      pv[u] = static_cast<uint32_t>(a);
      ps[u] = static_cast<uint32_t>(a >> 32);
      pv[u + 1] = static_cast<uint32_t>(b);
      ps[u + 1] = static_cast<uint32_t>(b >> 32);
    }
  }
  // Every word of a row <= rows carries its row tag?  A tree of integer ORs (an `ok = ok &&`
  // chain compiles to a serial chain of predicated compares).
  __device__ __forceinline__ bool block_ready(int r0, const uint32_t (&ps)[U]) const {
    const uint32_t exp0 = static_cast<uint32_t>(r0) << 16;
    uint32_t d[U];
#pragma unroll
    for (int u = 0; u < U; ++u) d[u] = ps[u] ^ (exp0 + (static_cast<uint32_t>(u) << 16));
    if (r0 + U - 1 > rows) {
#pragma unroll
      for (int u = 0; u < U; ++u) d[u] = (r0 + u <= rows) ? d[u] : 0u;
    }
#pragma unroll
    for (int w = 1; w < U; w *= 2)
#pragma unroll
      for (int u = 0; u + w < U; u += 2 * w) d[u] |= d[u + w];
    return (d[0] >> 16) == 0u || (WF_NW7_ABL & 2);
  }
  // (re)load until ready
  __device__ __forceinline__ bool wait_block(int r0, uint32_t (&pv)[U], uint32_t (&ps)[U]) {
    wd.start();
    for (;;) {
      ++retries;
      issue_block(r0, pv, ps);
      if (block_ready(r0, ps)) return true;
      if (wd.expired(L)) return false;
    }
  }
  __device__ __forceinline__ void finish_block(uint32_t (&ps)[U]) const {
    if constexpr (!PRMT) {
#pragma unroll
      for (int u = 0; u < U; ++u) ps[u] &= 0xffffu;
    }
  }

  unsigned retries = 0;
  int seen_next = 0;   // last observed consumption of the ring this warp writes
  __device__ __forceinline__ bool wait_ctr(const int* ctr, int need) {
    if (seen_next >= need) return true;
    wd.start();
    for (;;) {
      seen_next = lds_vol_i(ctr);
      if (seen_next >= need) return true;
      if (wd.expired(L)) return false;
      __nanosleep(32);
    }
  }

  template <bool EDGE>
  __device__ __forceinline__ void block(int t0, const uint32_t (&pv)[U], const uint32_t (&ps)[U], int32_t& Win,
                                        uint32_t& Sin) {
    const int src_lane = (lane + 31) & 31;
    const int r31_0 = t0 - 30;                 // lane 31's row at step t0
    unsigned long long* nslot = nextll + ll7_slot(r31_0);   // contiguous for the block
    const uint32_t hi0 = static_cast<uint32_t>(r31_0) << 16;   // LL tag of lane 31's row at u = 0
#pragma unroll
    for (int u = 0; u < U; ++u) {
      const int row = t0 + u - lane + 1;
      // the next row's selector does not depend on this row: rotate it first
      const uint32_t Snext = __shfl_sync(0xffffffffu, (lane == 31) ? ps[u] : Sin, src_lane);
      int32_t H[K];
      cells(Win, H);
      // rotate: lanes 0..30 pass their east value right; lane 31 passes lane 0's next west
      // input (row t0+u+2) around
      const int32_t Wnext = __shfl_sync(0xffffffffu, (lane == 31) ? static_cast<int32_t>(pv[u]) : H[K - 1], src_lane);
      bool active = true;
      if constexpr (EDGE) {
        active = row >= 1 && row <= rows;
        prevW = active ? Win : prevW;
#pragma unroll
        for (int m = 0; m < K; ++m) Np[m] = active ? H[m] : Np[m];
        if (active) stage_store(row, H);
      } else {
        prevW = Win;
#pragma unroll
        for (int m = 0; m < K; ++m) Np[m] = H[m];
        stage_store(row, H);
      }
      // lane 31: east value of row r31_0+u into the next warp's / the band's east LL ring
      sts_u64_if(lane == 31 && active, nslot + u,
                 (static_cast<unsigned long long>((hi0 + (static_cast<uint32_t>(u) << 16)) | (Sin & 0xffffu)) << 32) |
                     static_cast<uint32_t>(H[K - 1]));
      prep(Snext);
      Win = Wnext;
      Sin = Snext;
    }
  }

  __device__ __forceinline__ bool run() {
    const int T = rows + 31;
    if (L.trace && warp == 0 && lane == 0) L.trace[size_t(band) * kTraceSlots] = globaltimer();
    // lane 0's first west word (row 1)
    int32_t Win = 0;
    uint32_t Sin = 0;
    {
      const unsigned long long* p = myll + ll7_slot(1);
      wd.start();
      for (;;) {
        const unsigned long long w = lds_vol(p);
        if (static_cast<uint32_t>(w >> 48) == 1u) {
          if (lane == 0) {
            Win = static_cast<int32_t>(static_cast<uint32_t>(w));
            Sin = static_cast<uint32_t>(w >> 32) & 0xffffu;
          }
          break;
        }
        if (wd.expired(L)) return false;
      }
    }
    prep(Sin);
    // WF_TRACE phase profile (lane 0 of warps 0..3): SM cycles in [west wait, ring / staging
    // back-pressure, block compute, publish]
    const bool prof = L.trace != nullptr && lane == 0 && warp < 4;
    long long ph[4] = {0, 0, 0, 0};
    long long tc = prof ? clock64() : 0;
    auto tick = [&](int i) {
      if (prof) {
        const long long n = clock64();
        ph[i] += n - tc;
        tc = n;
      }
    };
    if (L.trace && warp == 0 && lane == 0) L.trace[size_t(band) * kTraceSlots + 42] = clock64();
    int blk = 0;
    uint32_t pv[U], ps[U];
    issue_block(2, pv, ps);
    if (!block_ready(2, ps) && !wait_block(2, pv, ps)) return false;
    for (int t0 = 0; t0 < T; t0 += U, ++blk) {
      tick(3);
      finish_block(ps);
      if (lane == 0) sts_vol_i(sm.rprog + warp, t0 + U + 1);     // rows <= t0+U+1 of my ring consumed
      tick(0);
      // the next ring's slots of lane 31's rows (t0-30 ..) must be free
      if (!wait_ctr(sm.rprog + warp + 1, t0 - 30 + U - 1 - kLL7)) return false;
      // staging slots: all but the last TMA group must have finished reading
      if constexpr (WF_NW7_PUB == 0) {
        if (lane == 0) bulk_wait_read<1>();
        __syncwarp();
      }
      tick(1);
      if (t0 >= 32 && t0 + U <= rows) block<false>(t0, pv, ps, Win, Sin);
      else block<true>(t0, pv, ps, Win, Sin);
      tick(2);
      // prefetch the next block's west words; their latency hides behind the write-back
      uint32_t nv[U], ns[U];
      issue_block(t0 + U + 2, nv, ns);
      if constexpr (WF_NW7_PUB == 1) {
        // write back lane 31's rows of this block (every lane is past them): row by row,
        // 32*K contiguous int32 per warp (coalesced 16-B stores)
        if (!(WF_NW7_ABL & 1)) {
          const int r31_0 = t0 - 30;
          __syncwarp();
          if (r31_0 >= 1 && r31_0 + U - 1 <= rows) {
#pragma unroll
            for (int u = 0; u < U; ++u) write_row(r31_0 + u);
          } else {
            const int lo = max(r31_0, 1), hi = min(r31_0 + U - 1, rows);
            for (int r = lo; r <= hi; ++r) write_row(r);
          }
        }
      } else if (((blk & 1) || t0 + U >= T) && !(WF_NW7_ABL & 1)) {
        // publish lane 31's rows of the last two blocks (all lanes are past them): one TMA box
        const int r31_0 = (blk & 1) ? t0 - U - 30 : t0 - 30;
        const int r31_last = min(t0 - 30 + U - 1, rows);
        if (r31_last >= 1) {
          fence_proxy_async_smem();
          __syncwarp();
          if (r31_0 >= 1) {
            if (lane == 0) {
              tma_store_2d(tmap, stage_w_s + ((r31_0 + kOff) & (R - 1)) * ROWB, wcol, r31_0 - 1);
              bulk_commit();
            }
          } else {
            for (int r = 1; r <= r31_last; ++r) write_row(r);
          }
        }
      }
      if (t0 + U < T) {
        if (!block_ready(t0 + U + 2, ns) && !wait_block(t0 + U + 2, nv, ns)) return false;
#pragma unroll
        for (int u = 0; u < U; ++u) {
          pv[u] = nv[u];
          ps[u] = ns[u];
        }
      }
    }
    if (lane == 0) {
      if constexpr (WF_NW7_PUB == 0) bulk_wait_all();
      sts_vol_i(sm.rprog + warp, rows + kLL7 + 64);
    }
    if (prof) {
      for (int i = 0; i < 4; ++i) L.trace[size_t(band) * kTraceSlots + 48 + 4 * warp + i] = ph[i];
      L.trace[size_t(band) * kTraceSlots + 36 + warp] = retries;
    }
    if (L.trace && warp == 0 && lane == 0) {
      L.trace[size_t(band) * kTraceSlots + kTraceRows] = globaltimer();
      L.trace[size_t(band) * kTraceSlots + 43] = clock64();
    }
    return true;
  }
};

// Feeder warp: warp 0's west words (column-0 boundary, or the band's global LL ring filled by
// the previous band / slab), with the row's score selector computed from x_i.
template <int K, int WARPS, int U, bool PRMT>
__device__ __forceinline__ bool nw7_feeder(const SweepLaunch& L, const Nw7Smem<K, WARPS, U>& sm, int band, int lane) {
  const int rows = L.rows;
  const uint8_t* x = static_cast<const uint8_t*>(L.row_in);
  const bool boundary = L.first_slab && band == 0;
  const unsigned long long* src = L.edge + size_t(band) * edge_stride(rows);
  unsigned long long* ring = sm.ll;   // warp 0's ring
  int feed = 1;
  int seen_rd = 0;
  unsigned iters = 0, bp = 0, empty = 0;
  Watchdog wd;
  wd.start();
  while (feed <= rows) {
    ++iters;
    const int need = feed + 63 - kLL7;   // slot reuse: warp 0 has consumed those rows
    if (seen_rd < need) {
      seen_rd = lds_vol_i(sm.rprog + 0);
      if (seen_rd < need) {
        ++bp;
        if (wd.expired(L)) return false;
        __nanosleep(32);
        continue;
      }
    }
    int32_t v[2];
    uint32_t s[2];
    bool ok[2];
#pragma unroll
    for (int h = 0; h < 2; ++h) {
      const int r = feed + h * 32 + lane;
      ok[h] = true;
      v[h] = 0;
      s[h] = 0;
      if (r <= rows) {
        const uint32_t xc = __ldg(x + (r - 1));
        s[h] = PRMT ? xc * 0x1111u + 0x8880u : xc;
        if (boundary) {
          v[h] = r * L.gap;   // H[r][0] = r*g
        } else {
          const unsigned long long w = ld_relaxed_sys(src + r);
          v[h] = static_cast<int32_t>(static_cast<uint32_t>(w));
          ok[h] = static_cast<uint32_t>(w >> 32) == L.epoch;
        }
      }
    }
    const unsigned m0 = __ballot_sync(0xffffffffu, ok[0]);
    const unsigned m1 = __ballot_sync(0xffffffffu, ok[1]);
    int n = (m0 == 0xffffffffu) ? 32 + (__ffs(~m1) ? __ffs(~m1) - 1 : 32) : __ffs(~m0) - 1;
    if (feed + n > rows + 1) n = rows + 1 - feed;
    if (n > 0) {
#pragma unroll
      for (int h = 0; h < 2; ++h) {
        const int r = feed + h * 32 + lane;
        if (r < feed + n) sts_u64(ring + ll7_slot(r), ll7(v[h], s[h], r));
      }
      feed += n;
      wd.start();
      if (feed > rows && !L.first_slab && band == 0 && L.ack_prev) {
        __syncwarp();
        if (lane == 0) st_relaxed_sys_u32(L.ack_prev, L.epoch);   // predecessor slab may reuse this ring
      }
    } else {
      ++empty;
      if (wd.expired(L)) return false;
      __nanosleep(32);
    }
  }
  if (L.trace && lane == 0) {
    L.trace[size_t(band) * kTraceSlots + 44] = iters;
    L.trace[size_t(band) * kTraceSlots + 45] = bp;
    L.trace[size_t(band) * kTraceSlots + 46] = empty;
  }
  return true;
}

// Forwarder warp: the band's east edge (ring WARPS, written per row by lane 31 of the last
// compute warp) to the next band's global LL ring, or -- last band of a slab -- to the next
// slab's band-0 ring through a peer (NVLink) mapping.  Coalesced 8-byte LL stores.
template <int K, int WARPS, int U>
__device__ __forceinline__ bool nw7_forwarder(const SweepLaunch& L, const Nw7Smem<K, WARPS, U>& sm, int band, int lane) {
  const int rows = L.rows;
  const bool to_next_slab = band + 1 >= L.nbands;
  unsigned long long* dst = to_next_slab ? L.next_edge : L.edge + size_t(band + 1) * edge_stride(rows);
  const unsigned long long* ring = sm.ll + size_t(WARPS) * kLL7;
  Watchdog wd;
  if (dst && to_next_slab && L.ack_self) {   // the next slab must have drained its ring (previous run)
    wd.start();
    for (;;) {
      const unsigned a = ld_relaxed_sys_u32(L.ack_self);
      if (static_cast<int>(a - (L.epoch - 1u)) >= 0) break;
      if (wd.expired(L)) return false;
      __nanosleep(64);
    }
  }
  int fwd = 1;
  wd.start();
  while (fwd <= rows) {
    const int r = fwd + lane;
    bool ok = true;
    unsigned long long w = 0;
    if (r <= rows) {
      w = lds_vol(ring + ll7_slot(r));
      ok = static_cast<uint32_t>(w >> 48) == (static_cast<uint32_t>(r) & 0xffffu);
    }
    const unsigned m = __ballot_sync(0xffffffffu, ok);
    int n = (m == 0xffffffffu) ? 32 : __ffs(~m) - 1;
    if (fwd + n > rows + 1) n = rows + 1 - fwd;
    if (n > 0) {
      if (dst && lane < n) st_relaxed_sys(dst + r, ll_pack(static_cast<uint32_t>(w), L.epoch));
      fwd += n;
      __syncwarp();
      if (lane == 0) sts_vol_i(sm.rprog + WARPS, fwd - 1);
      wd.start();
    } else {
      if (wd.expired(L)) return false;
      __nanosleep(16);
    }
  }
  return true;
}

template <int K, int WARPS, int U, bool PRMT, int FORM>
__global__ void __launch_bounds__((WARPS + 2) * 32)
    nw7_kernel(const SweepLaunch L, const __grid_constant__ CUtensorMap tmap) {
  using S = Nw7Smem<K, WARPS, U>;
  extern __shared__ __align__(16) unsigned char nw7_smem_raw[];
  const S sm(nw7_smem_raw);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  for (int band = blockIdx.x; band < L.nbands; band += gridDim.x) {
    for (int i = threadIdx.x; i < (WARPS + 1) * kLL7; i += blockDim.x) sm.ll[i] = 0ull;
    if (threadIdx.x < 64) sm.rprog[threadIdx.x] = 0;
    __syncthreads();
    if (warp == WARPS) {
      nw7_feeder<K, WARPS, U, PRMT>(L, sm, band, lane);
    } else if (warp == WARPS + 1) {
      nw7_forwarder<K, WARPS, U>(L, sm, band, lane);
    } else {
      Nw7Warp<K, WARPS, U, PRMT, FORM> w(L, &tmap, sm, band, warp, lane);
      w.run();
    }
    __syncthreads();
    if (run_failed(L)) return;
  }
}

cudaError_t encode_plane_map(CUtensorMap* m, const SweepLaunch& L, int box_cols, int box_rows);

namespace {

int form_env() {
  const char* e = getenv("WF_NW7_FORM");
  return (e && e[0] == '1') ? 1 : 0;
}

template <int K, int W, int U, int FORM>
cudaError_t launch_nw7_f(const SweepLaunch& L, cudaStream_t s, size_t smem) {
  CUtensorMap tmap;
  cudaError_t e = encode_plane_map(&tmap, L, 32 * K, 2 * U);
  if (e != cudaSuccess) return e;
  auto kfn = (L.alphabet >= 1 && L.alphabet <= 8) ? nw7_kernel<K, W, U, true, FORM> : nw7_kernel<K, W, U, false, FORM>;
  e = cudaFuncSetAttribute(kfn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  kfn<<<L.grid, (W + 2) * 32, smem, s>>>(L, tmap);
  return cudaGetLastError();
}

template <int K, int W, int U>
cudaError_t launch_nw7(const SweepLaunch& L, cudaStream_t s, size_t smem) {
  return form_env() ? launch_nw7_f<K, W, U, 1>(L, s, smem) : launch_nw7_f<K, W, U, 0>(L, s, smem);
}

// One band per SM: the shared-memory request is padded past half an SM's capacity, so the
// block scheduler cannot stack two bands on one SM while others idle (WF_NW7_PAD=0: off)
size_t nw7_smem(size_t need) {
  const char* e = getenv("WF_NW7_PAD");
  if (e && e[0] == '0') return need;
  return need > 120 * 1024 ? need : 120 * 1024;
}

template <int K, int W>
Variant make_nw7() {
  constexpr int U = 16;
  using S = Nw7Smem<K, W, U>;
  return Variant{WF_FN_SEQCMP, 0, K, W, 1, (W + 2) * 32, nw7_smem(S::bytes),
                 reinterpret_cast<const void*>(nw7_kernel<K, W, U, true, 0>), &launch_nw7<K, W, U>, 7};
}

}  // namespace

const Variant* nw7_table(size_t* n) {
#ifdef WF_MIN_VARIANTS
  static const Variant v[] = {make_nw7<4, 2>()};
#else
  static const Variant v[] = {make_nw7<4, 1>(), make_nw7<4, 2>(), make_nw7<2, 2>(), make_nw7<2, 4>(),
                              make_nw7<8, 1>()};
#endif
  *n = sizeof(v) / sizeof(v[0]);
  return v;
}

}  // namespace wfk
