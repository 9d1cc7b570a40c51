// wf_syn.cu -- the synthetic application's band sweep (Sec. 3.1.1;
// cell in wf_cells.cuh::PolSyn, readings R4-R6 of DESIGN.md), sm_100a.
//
// Same band / lane / skew model as the other sweeps (wf_sweep.cuh): a persistent CTA owns a
// band of WARPS*32*K columns and sweeps all its rows; lane l owns K adjacent columns and at
// step t is on row t - l + 1, its west input arriving from lane l-1 by __shfl_up_sync.
// What this kernel adds for the synthetic cell (tsize-deep fp32 FMA chains, 2 + dsize
// output planes):
//  * The row input u_i travels WITH the west words (one more LL word per row, then lane to
//    lane by shuffle): no global load in the row loop.
//  * Lane 0's west words for row t+2 are loaded (broadcast LDS) one step ahead and their
//    tags checked with an OR tree, so the shared-memory latency is off the FMA chain.
//  * Outputs go to a per-warp, per-plane staging ring and leave as one TMA 2-D tensor store
//    per plane and U-row block (every output byte written once, coalesced).
//  * Lane 31 hands its east words to the next warp through a shared LL ring (tag = row), the
//    band's last warp to the next band / slab through the global LL ring (tag = epoch).
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

constexpr int kSynLL = 128;   // rows per shared west LL ring (power of 2)
// Block sizes, measured on C2 / C5a-c:
//  * TMA write-back window UT: 32 rows amortise the proxy fence; 16 rows when the planes are
//    many (dsize > 2), so that 4 one-warp CTAs still fit per SM (512 bands at dim 16384).
//  * west hand-off block UB: the hand-off lag is UB + 31 steps per warp; with deep cells
//    (large tsize) a step is expensive and small blocks win, with light cells the per-block
//    cost dominates: UB = 16 / 8 / 4 for tsize x dsize < 40 / < 1000 (or runtime) / >= 1000.
__host__ __device__ constexpr int syn_ut(int ds) { return ds <= 2 ? 32 : 16; }
#ifndef WF_SYN_UB_LIGHT
#define WF_SYN_UB_LIGHT 16   // experiments: hand-off block of light cells (tsize x dsize < 40)
#endif
#ifndef WF_SYN_UB_MID
#define WF_SYN_UB_MID 8      // experiments: hand-off block of medium cells (< 1000, or runtime tsize)
#endif
__host__ __device__ constexpr int syn_ub(int ts, int ds) {
  return ts == 0 ? WF_SYN_UB_MID
                 : (ts * (ds > 0 ? ds : 1) >= 1000 ? 4 : ts * (ds > 0 ? ds : 1) >= 40 ? WF_SYN_UB_MID : WF_SYN_UB_LIGHT);
}

struct SynMaps {
  CUtensorMap m[WF_MAX_PLANES];
};

// Global LL ring record of a row: NF 8-byte words (value | run-epoch tag) padded to a multiple
// of 4 words, so the band's last lane writes each row with 32-byte stores that cover whole L2
// sectors (no fill read of the sector; the consumer discards consumed lines, so the ring costs
// no DRAM traffic -- profiles/r02_c5a_traffic.txt).  The host sizes the rings with the same
// padding (wf_api.cpp: ring_words).
__host__ __device__ constexpr int syn_ring_words(int nf) { return (nf + 3) & ~3; }

template <int DS, int K, int WARPS>
struct SynSmem {
  static constexpr int NF = 2 + DS;         // output planes / west words per row
  static constexpr int NFP = syn_ring_words(NF);   // global ring words per row
  static constexpr int NWD = NF + 1;        // + the row input u_i
  static constexpr int U = syn_ut(DS);
  // staging rows alive: skew 31 + the TMA window being filled + the window whose TMA store
  // may still be reading
  static constexpr int R = (2 * U + 31) <= 64 ? 64 : 128;
  static_assert(2 * U + 31 <= R, "staging ring too small");
  static constexpr int ROWB = 32 * K * 4;
  static constexpr size_t stage_bytes = size_t(WARPS) * NF * R * ROWB;
  static constexpr size_t ll_bytes = size_t(WARPS) * kSynLL * NWD * 4;
  static constexpr size_t bytes = 1024 + stage_bytes + ll_bytes + 64 * 4;
  unsigned char* stage;     // [WARPS][NF][R][32K] u32, 1024-byte aligned (TMA sources)
  uint32_t* ll;             // [WARPS][kSynLL][NWD]: ring w = west words (+ u_i) of warp w
  int* rprog;               // rprog[w]: rows of ring w consumed by warp w
  int* wprog;               // wprog[w]: rows of ring w published by its producer
  __device__ __forceinline__ explicit SynSmem(unsigned char* raw) {
    const uint32_t a = static_cast<uint32_t>(__cvta_generic_to_shared(raw));
    unsigned char* base = raw + ((1024u - (a & 1023u)) & 1023u);
    stage = base;
    ll = reinterpret_cast<uint32_t*>(base + stage_bytes);
    rprog = reinterpret_cast<int*>(base + stage_bytes + ll_bytes);
    wprog = rprog + 32;
  }
  __device__ __forceinline__ uint32_t* slot(int w, int row) const {
    return ll + (size_t(w) * kSynLL + (row & (kSynLL - 1))) * NWD;
  }
};

#ifndef WF_SYN_STEP_WAIT
// Heavy cells (tsize x dsize >= 1000, UB = 4): a compute warp waits for its west words row by row
// (a cached copy of the producer's counter, re-read only when it does not cover the step's row)
// instead of for the whole UB-row block, so the band-to-band lag loses up to UB - 1 steps
// (C5c 78.28 -> 76.19 ms).  Light cells keep the block wait: there a step is short and the
// per-step check at the producer's heels costs more than it saves (C5a 3.88 -> 5.55 ms); so do
// many-plane heavy cells (C5d 129.6 -> 131.8 ms with it); profiles/r02_syn_lds_ab.txt.
// 0 = never, 1 = heavy cells with dsize <= 2, 2 = always (experiments).
#define WF_SYN_STEP_WAIT 1
#endif
__device__ __forceinline__ void sts_u32_pred(bool p, uint32_t* a, uint32_t v) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q st.volatile.shared.u32 [%0], %1; }" ::"r"(
                   static_cast<uint32_t>(__cvta_generic_to_shared(a))),
               "r"(v), "r"(static_cast<int>(p))
               : "memory");
}
#ifndef WF_SYN_ST
#define WF_SYN_ST 1   // band-to-band LL store: 0 st.relaxed.sys, 1 st.relaxed.gpu, 2 weak st.global
#endif
__device__ __forceinline__ uint32_t lds_vol_u32(const uint32_t* p) { return *reinterpret_cast<const volatile uint32_t*>(p); }
__device__ __forceinline__ void stg_sys_u64_pred(bool p, unsigned long long* a, unsigned long long v) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q st.relaxed.sys.global.u64 [%0], %1; }" ::"l"(a), "l"(v),
               "r"(static_cast<int>(p))
               : "memory");
}
// 32-byte strong store of 4 LL words (STG.E.ENL2.256): whole L2 sectors
__device__ __forceinline__ void stg_sys_v4_pred(bool p, unsigned long long* a, unsigned long long w0, unsigned long long w1,
                                                unsigned long long w2, unsigned long long w3) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %5, 0; @q st.relaxed.sys.global.v4.b64 [%0], {%1, %2, %3, %4}; }" ::"l"(a),
               "l"(w0), "l"(w1), "l"(w2), "l"(w3), "r"(static_cast<int>(p))
               : "memory");
}
__device__ __forceinline__ void stg_gpu_u64_pred(bool p, unsigned long long* a, unsigned long long v) {
#if WF_SYN_ST == 0
  stg_sys_u64_pred(p, a, v);
#elif WF_SYN_ST == 1
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q st.relaxed.gpu.global.u64 [%0], %1; }" ::"l"(a), "l"(v),
               "r"(static_cast<int>(p))
               : "memory");
#else
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q st.global.u64 [%0], %1; }" ::"l"(a), "l"(v),
               "r"(static_cast<int>(p))
               : "memory");
#endif
}

// PW >= 0: plane-split warp (impl 8, one column warp per band): the CTA runs DS compute warps
// on the SAME 32 columns, warp PW computing float item d = PW (warp 0 also the two int fields).
// The items of a cell are independent given (N, W, NW, u_i, v_j) (R5), so each warp's tsize
// chain is one item deep instead of DS: the step is bound by one FMA chain's latency, not by
// DS x tsize FFMA issues of one warp.
template <int DS, int K, int WARPS, int TS, int PW = -1>
struct SynWarp {
  using P = PolSyn<DS>;
  using S = SynSmem<DS, K, WARPS>;
  static constexpr int NF = S::NF, NWD = S::NWD, U = S::U, R = S::R, ROWB = S::ROWB;
  static constexpr int kOff = 30 % U;   // lane 31's rows of a block occupy contiguous staging slots
  // does this warp compute / store / hand off field f
  __host__ __device__ static constexpr bool use(int f) { return PW < 0 || (f < 2 ? PW == 0 : f - 2 == PW); }
  static constexpr int kRd = PW < 0 ? 0 : PW;   // my consumed-rows counter: rprog[warp + kRd]

  // The synthetic cell of wf_cells.cuh::PolSyn (same single operations in the same order,
  // DESIGN.md R5/R11), with the tsize loop unrolled when tsize is a compile-time constant
  // (TS > 0; TS = 0: runtime trip count).
  __device__ __forceinline__ void cell(const uint32_t* N, const uint32_t* W, const uint32_t* NW, uint32_t ui,
                                       uint32_t vj, uint32_t* o) const {
    if (use(0)) {
      o[0] = static_cast<uint32_t>(max(max(static_cast<int>(N[0]), static_cast<int>(NW[0])), static_cast<int>(W[0])) + 1);
      o[1] = ((N[1] - NW[1]) + 1u) + W[1];
    } else {
      o[0] = 0u;
      o[1] = 0u;
    }
    if constexpr (DS > 0 && (PW < 0 || PW < DS)) {
      const float THIRD = __uint_as_float(0x3EAAAAABu);
      const float A = __uint_as_float(0x3F7FF000u);
      const float SCALE = __uint_as_float(0x39800000u);
      const float c = __fmul_rn(__fmul_rn(__uint_as_float(ui), __uint_as_float(vj)), SCALE);
      constexpr int D0 = PW < 0 ? 0 : PW, D1 = PW < 0 ? DS : PW + 1;   // my items [D0, D1)
      float x[DS];
#pragma unroll
      for (int d = 0; d < DS; ++d) x[d] = 0.f;
#pragma unroll
      for (int d = D0; d < D1; ++d)
        x[d] = __fmul_rn(__fadd_rn(__fadd_rn(__uint_as_float(N[2 + d]), __uint_as_float(NW[2 + d])),
                                   __uint_as_float(W[2 + d])),
                         THIRD);
      if constexpr (TS > 0) {
#pragma unroll 100
        for (int t = 0; t < TS; ++t) {
#pragma unroll
          for (int d = D0; d < D1; ++d) x[d] = __fmaf_rn(x[d], A, c);
        }
      } else {
        const int ts = pol.tsize;
#pragma unroll 4
        for (int t = 0; t < ts; ++t) {
#pragma unroll
          for (int d = D0; d < D1; ++d) x[d] = __fmaf_rn(x[d], A, c);
        }
      }
#pragma unroll
      for (int d = 0; d < DS; ++d) o[2 + d] = __float_as_uint(x[d]);
    }
  }

  const SweepLaunch& L;
  const P& pol;
  const SynMaps& maps;
  const S& sm;
  const int band, warp, lane;
  int rows;
  uint32_t cin[K];
  uint32_t Np[K][NF];
  uint32_t prevW[NF];
  int wcol;
  unsigned char* stage_w;
  Watchdog wd;

  __device__ __forceinline__ SynWarp(const SweepLaunch& L_, const P& pol_, const SynMaps& maps_, const S& sm_, int band_,
                                     int warp_, int lane_)
      : L(L_), pol(pol_), maps(maps_), sm(sm_), band(band_), warp(warp_), lane(lane_) {
    rows = L.rows;
    wcol = band * L.band_w + warp * 32 * K;
    const int jb = L.c0 + wcol + lane * K;   // 0-based global column of the lane's first column
#pragma unroll
    for (int m = 0; m < K; ++m) {
      const int j1 = jb + m + 1;
      const bool vc = (jb + m) < L.c1;
      cin[m] = vc ? pol.col_in(j1) : 0u;
      pol.top(vc ? j1 : 0, Np[m]);
    }
    pol.top(jb < L.c1 ? jb : 0, prevW);
    stage_w = sm.stage + size_t(warp) * NF * R * ROWB;
  }

  __device__ __forceinline__ void stage_store(bool p, int row, const uint32_t (&H)[K][NF]) const {
    const int slot = (row + kOff) & (R - 1);
#pragma unroll
    for (int f = 0; f < NF; ++f) {
      if (!use(f)) continue;
      uint32_t* dst = reinterpret_cast<uint32_t*>(stage_w + (size_t(f) * R + slot) * ROWB) + lane * K;
#pragma unroll
      for (int m = 0; m < K; ++m) sts_u32_pred(p, dst + m, H[m][f]);
    }
  }

  __device__ __forceinline__ void write_row(int r) const {
    const int jrel = wcol + lane * K;
    const int width = L.c1 - L.c0;
    const int slot = (r + kOff) & (R - 1);
#pragma unroll
    for (int f = 0; f < NF; ++f) {
      if (!use(f)) continue;
      const uint32_t* src = reinterpret_cast<const uint32_t*>(stage_w + (size_t(f) * R + slot) * ROWB) + lane * K;
      uint32_t* dst = static_cast<uint32_t*>(L.out[f]) + int64_t(r - 1) * L.pitch + jrel;
#pragma unroll
      for (int m = 0; m < K; ++m)
        if (jrel + m < width) dst[m] = src[m];
    }
  }

  // lane 0's west words + row input of row r (all lanes load: broadcast).  Plain loads: every
  // block starts after wait_ctr observed the producer's counter covering the block's rows and
  // fenced (__threadfence_block, also a compiler barrier), so the words are there and no load
  // can move above it; unlike volatile loads they need not stay in program order with the
  // step's shared stores (C5a 4.044 -> 3.876 ms, profiles/r02_syn_lds_ab.txt)
  __device__ __forceinline__ void issue(int r, uint32_t (&w)[NWD]) const {
    const uint32_t* p = sm.slot(warp, r);
#pragma unroll
    for (int i = 0; i < NWD; ++i) w[i] = (i == NF || use(i)) ? p[i] : 0u;
  }
  // wait until a shared progress counter reaches `need` (seen caches the last value)
  __device__ __forceinline__ bool wait_ctr(const int* ctr, int need, int& seen) {
    if (seen >= need) return true;
    wd.start();
    for (;;) {
      seen = lds_vol_i(ctr);
      if (seen >= need) {
        __threadfence_block();   // order the ring reads after the observed counter
        return true;
      }
      if (wd.expired(L)) return false;
    }
  }

  static constexpr bool kStepWait = WF_SYN_STEP_WAIT == 2 || (WF_SYN_STEP_WAIT == 1 && syn_ub(TS, DS) <= 4 && DS <= 2);

  template <bool EDGE, bool LAST>
  __device__ __forceinline__ bool block(int t0, uint32_t (&pre)[NWD], uint32_t (&q)[NF], uint32_t& qx,
                                        unsigned long long* gdst, bool to_peer, int& seen_w) {
    uint32_t* nring = LAST ? nullptr : sm.ll + size_t(warp + 1) * kSynLL * NWD;
    const bool glob = LAST && gdst != nullptr;
#pragma unroll
    for (int u = 0; u < syn_ub(TS, DS); ++u) {
      const int t = t0 + u;
      const int row = t - lane + 1;
      uint32_t Win[NF];
#pragma unroll
      for (int f = 0; f < NF; ++f) Win[f] = (lane == 0) ? pre[f] : q[f];
      const uint32_t xr = (lane == 0) ? pre[NF] : qx;
      if (kStepWait && u > 0 && t + 2 <= rows && seen_w < t + 2) {   // (u = 0: run() waited)
        if (!wait_ctr(sm.wprog + warp, t + 2, seen_w)) return false;
      }
      if (!EDGE || t + 2 <= rows) issue(t + 2, pre);   // next step's words: latency hides behind the cell
      bool active = true;
      if constexpr (EDGE) active = row >= 1 && row <= rows;
      // every lane evaluates (inactive lanes on don't-care inputs) -- no divergent branch
      uint32_t H[K][NF];
#pragma unroll
      for (int m = 0; m < K; ++m) {
        const uint32_t* NWm = (m == 0) ? prevW : Np[m - 1];
        const uint32_t* Wm = (m == 0) ? Win : H[m - 1];
        cell(Np[m], Wm, NWm, xr, cin[m], H[m]);
      }
#pragma unroll
      for (int f = 0; f < NF; ++f) {
        prevW[f] = active ? Win[f] : prevW[f];
#pragma unroll
        for (int m = 0; m < K; ++m) Np[m][f] = active ? H[m][f] : Np[m][f];
      }
      stage_store(active, row, H);
      // lane 31: east words of its row to the next warp's ring (+ u_i), or the next band's /
      // slab's global LL ring
      const bool pub = lane == 31 && active;
      if constexpr (!LAST) {
        uint32_t* sl = nring + (row & (kSynLL - 1)) * NWD;
#pragma unroll
        for (int f = 0; f < NF; ++f) sts_u32_pred(pub, sl + f, Np[K - 1][f]);
        sts_u32_pred(pub, sl + NF, xr);
      } else {
        // system scope: the next slab's ring may be a peer (NVLink) mapping; measured no slower
        // than gpu scope for the next band's ring on the same GPU
        unsigned long long* g = gdst + size_t(row) * S::NFP;
        (void)to_peer;
        if constexpr (PW < 0) {   // the whole record: 32-byte stores (full L2 sectors)
          const uint32_t ep = L.epoch;
#pragma unroll
          for (int c = 0; c < S::NFP; c += 4)
            stg_sys_v4_pred(pub && glob, g + c, ll_pack(c < NF ? Np[K - 1][c] : 0u, ep),
                            ll_pack(c + 1 < NF ? Np[K - 1][c + 1 < NF ? c + 1 : 0] : 0u, ep),
                            ll_pack(c + 2 < NF ? Np[K - 1][c + 2 < NF ? c + 2 : 0] : 0u, ep),
                            ll_pack(c + 3 < NF ? Np[K - 1][c + 3 < NF ? c + 3 : 0] : 0u, ep));
        } else {   // plane-split warps own some fields of the record
#pragma unroll
          for (int f = 0; f < NF; ++f)
            if (use(f)) stg_sys_u64_pred(pub && glob, g + f, ll_pack(Np[K - 1][f], L.epoch));
        }
      }
#pragma unroll
      for (int f = 0; f < NF; ++f) q[f] = use(f) ? __shfl_up_sync(0xffffffffu, Np[K - 1][f], 1) : 0u;
      qx = __shfl_up_sync(0xffffffffu, xr, 1);
    }
    return true;
  }

  __device__ __forceinline__ bool run() {
    const int T = rows + 31;
    const bool last = warp + 1 == WARPS;
    if (last && band + 1 >= L.nbands && L.next_edge && L.ack_self) {   // next slab drained its ring
      wd.start();
      for (;;) {
        const unsigned a = ld_relaxed_sys_u32(L.ack_self);
        if (static_cast<int>(a - (L.epoch - 1u)) >= 0) break;
        if (wd.expired(L)) return false;
        __nanosleep(64);
      }
    }
    unsigned long long* gdst = nullptr;
    if (last) gdst = (band + 1 < L.nbands) ? L.edge + size_t(band + 1) * edge_stride(rows) * S::NFP : L.next_edge;
    const bool to_peer = band + 1 >= L.nbands;
    int seen_w = 0, seen_r = 0;
    uint32_t pre[NWD];
    if (!wait_ctr(sm.wprog + warp, 1, seen_w)) return false;
    issue(1, pre);
    if (L.trace && lane == 0) {
      L.trace[size_t(band) * kTraceSlots + 44 + warp] = globaltimer();   // first row available
      if (warp == 0) L.trace[size_t(band) * kTraceSlots] = globaltimer();
    }
    uint32_t q[NF], qx = 0;
#pragma unroll
    for (int f = 0; f < NF; ++f) q[f] = 0u;
    const uint32_t stage_s = static_cast<uint32_t>(__cvta_generic_to_shared(stage_w));
    constexpr int UB = syn_ub(TS, DS);
    static_assert(U % UB == 0, "hand-off blocks tile the write-back window");
    for (int t0 = 0; t0 < T; t0 += UB) {
      // this block reads rows t0+2 .. t0+UB+1 of my ring (row t0+1 is already in pre)
      if (!wait_ctr(sm.wprog + warp, min(kStepWait ? t0 + 2 : t0 + UB + 1, rows), seen_w)) return false;
      if (lane == 0) sts_vol_i(sm.rprog + warp + kRd, t0 + 1);   // rows <= t0+1 of my ring consumed
      // lane 31 writes rows t0-30 .. t0-31+UB into the next ring: their slots must be free
      if (!last && !wait_ctr(sm.rprog + warp + 1, t0 - 31 + UB - kSynLL, seen_r)) return false;
      if (t0 % U == 0) {
        if (lane == 0) bulk_wait_read<1>();                // staging slots of 2 windows ago are free
        __syncwarp();
      }
      const bool steady = t0 >= 32 && t0 + UB + 1 <= rows;
      bool ok;
      if (last) {
        if (steady) ok = block<false, true>(t0, pre, q, qx, gdst, to_peer, seen_w);
        else ok = block<true, true>(t0, pre, q, qx, gdst, to_peer, seen_w);
      } else {
        if (steady) ok = block<false, false>(t0, pre, q, qx, gdst, to_peer, seen_w);
        else ok = block<true, false>(t0, pre, q, qx, gdst, to_peer, seen_w);
      }
      if (!ok) return false;
      wf_jitter(15);
      // publish lane 31's rows of the block to the next warp (one fence per block)
      const int r31_last = min(t0 + UB - 31, rows);
      if (!last && r31_last >= 1 && lane == 31) {
        __threadfence_block();
        sts_vol_i(sm.wprog + warp + 1, r31_last);
      }
      // write back lane 31's rows of the U-row window (every lane is past them): one TMA box
      // per plane when the window is complete (or the sweep ends)
      const bool win_end = (t0 + UB) % U == 0 || t0 + UB >= T;
      if (win_end && r31_last >= 1) {
        const int w0 = ((t0 + UB - 1) / U) * U;            // window start step (multiple of U)
        const int r31_0 = w0 - 30;                          // its first lane-31 row
        fence_proxy_async_smem();
        __syncwarp();
        if (r31_0 >= 1) {
          if (lane == 0) {
#pragma unroll
            for (int f = 0; f < NF; ++f)
              if (use(f)) tma_store_2d(&maps.m[f], stage_s + (f * R + ((r31_0 + kOff) & (R - 1))) * ROWB, wcol, r31_0 - 1);
            bulk_commit();
          }
        } else {
          for (int r = 1; r <= r31_last; ++r) write_row(r);
        }
      }
    }
    if (lane == 0) {
      bulk_wait_all();
      sts_vol_i(sm.rprog + warp + kRd, rows + kSynLL + 64);
    }
    if (L.trace && lane == 0) {
      L.trace[size_t(band) * kTraceSlots + 52 + warp] = globaltimer();
      if (warp == 0) L.trace[size_t(band) * kTraceSlots + kTraceRows] = globaltimer();
    }
    return true;
  }
};

// Feeder warp: warp 0's west words (column-0 boundary planes, or the band's global LL ring
// written by the previous band / slab) plus u_i, as row-tagged LL words in shared memory.
// Feeder back-off between LL polls: spin for few planes (C5a 4.114 -> 4.075 ms, C2 -0.4 %),
// 64 ns for many planes (C5b +0.2 % when spinning); profiles/r01_syn_feed_ab.txt.
// WF_SYN_FEED_NS >= 0 forces it (experiments).
#ifndef WF_SYN_FEED_NS
#define WF_SYN_FEED_NS -1
#endif
__host__ __device__ constexpr unsigned syn_feed_ns(int ds) {
  return WF_SYN_FEED_NS >= 0 ? unsigned(WF_SYN_FEED_NS) : (ds <= 2 ? 0u : 64u);
}
#ifndef WF_SYN_FEED_WIN
// How the feeder polls its band's ring (profiles/r02_c5a_traffic.txt, same-box A/Bs):
//   0 = one 8-byte load per LL word, 32 rows per poll (C5a: fastest, 3.652 ms);
//   2 = 32-byte loads per record, 32 rows (C5b 7.455 -> 7.288 ms; C5a 3.788 ms);
//   1 = 32-byte loads and an adaptive window (rows delivered last time + 8, at most 32): fewer
//       polls of not-yet-written rows (C5a reads 267 -> 160 MB) but C5a 3.695 -> 3.876 ms.
//  -1 (default) = 2 for 8-word records (dsize >= 3), 0 otherwise.
#define WF_SYN_FEED_WIN -1
#endif
__device__ __forceinline__ void ldg_sys_v4(const unsigned long long* a, unsigned long long (&w)[4]) {
  asm volatile("ld.relaxed.sys.global.v4.b64 {%0, %1, %2, %3}, [%4];" : "=l"(w[0]), "=l"(w[1]), "=l"(w[2]), "=l"(w[3])
               : "l"(a)
               : "memory");
}
#ifndef WF_SYN_DISCARD
// 1: the feeder drops each fully consumed 128-byte line of its band's inbound LL ring from L2
// without write-back (discard.global.L2): the words are dead once copied to shared memory, so the
// ring costs no DRAM traffic (C5a: 1.106x -> ~1.0x algorithmic, profiles/ncu_traffic.json)
#define WF_SYN_DISCARD 1
#endif
__device__ __forceinline__ void discard_l2_line(const void* p) {
  asm volatile("discard.global.L2 [%0], 128;" ::"l"(p) : "memory");
}
template <int DS, int K, int WARPS, int NPW = 1>
__device__ __forceinline__ bool syn_feeder(const SweepLaunch& L, const PolSyn<DS>& pol, const SynSmem<DS, K, WARPS>& sm,
                                           int band, int lane) {
  using S = SynSmem<DS, K, WARPS>;
  constexpr int NF = S::NF;
  const int rows = L.rows;
  const bool boundary = L.first_slab && band == 0;
  constexpr int NFP = S::NFP;
  const unsigned long long* src = L.edge + size_t(band) * edge_stride(rows) * NFP;
  // next ring line to discard: the first 128-byte line that starts at or after row 1's words (a
  // line below it may hold the previous band's ring, which another feeder still reads)
  uintptr_t disc = (reinterpret_cast<uintptr_t>(src + size_t(1) * NFP) + 127) & ~uintptr_t(127);
  int feed = 1, seen = 0;
  constexpr int kFeed = WF_SYN_FEED_WIN >= 0 ? WF_SYN_FEED_WIN : (NFP >= 8 ? 2 : 0);
  int win = 32;   // rows polled (kFeed 1)
  Watchdog wd;
  wd.start();
  while (feed <= rows) {
    wf_jitter(14);
    const int need = feed + 31 - kSynLL;   // slot reuse: warp 0 has consumed those rows
    if (seen < need) {
      seen = lds_vol_i(sm.rprog + 0);
#pragma unroll
      for (int p = 1; p < NPW; ++p) seen = min(seen, lds_vol_i(sm.rprog + p));   // plane-split readers
      if (seen < need) {
        if (wd.expired(L)) return false;
        __nanosleep(64);
        continue;
      }
    }
    const int r = feed + lane;
    uint32_t v[NF];
    bool ok = true;
    uint32_t xr = 0;
    if (r <= rows) {
      xr = pol.row_in(r);
      if (boundary) {
        pol.left(r, v);
      } else if (kFeed) {
        if (lane < win) {
#pragma unroll
          for (int c = 0; c < NFP; c += 4) {
            unsigned long long w[4];
            ldg_sys_v4(src + size_t(r) * NFP + c, w);
#pragma unroll
            for (int k = 0; k < 4; ++k)
              if (c + k < NF) {
                v[c + k] = static_cast<uint32_t>(w[k]);
                ok = ok && static_cast<uint32_t>(w[k] >> 32) == L.epoch;
              }
          }
        } else {
          ok = false;
        }
      } else {
#pragma unroll
        for (int f = 0; f < NF; ++f) {
          const unsigned long long w = ld_relaxed_sys(src + size_t(r) * NFP + f);
          v[f] = static_cast<uint32_t>(w);
          ok = ok && static_cast<uint32_t>(w >> 32) == L.epoch;
        }
      }
    }
    const unsigned m = __ballot_sync(0xffffffffu, ok);
    int n = (m == 0xffffffffu) ? 32 : __ffs(~m) - 1;
    if (kFeed == 1) win = min(32, max(8, n + 8));
    if (feed + n > rows + 1) n = rows + 1 - feed;
    if (n > 0) {
      if (lane < n) {
        uint32_t* sl = sm.slot(0, r);
#pragma unroll
        for (int f = 0; f < NF; ++f) sl[f] = v[f];
        sl[NF] = xr;
      }
      __syncwarp();
      __threadfence_block();
      feed += n;
      if (lane == 0) sts_vol_i(sm.wprog + 0, feed - 1);
      if (WF_SYN_DISCARD && !boundary) {
        // every line wholly below the consumed frontier (rows < feed), one line per lane
        const uintptr_t end = reinterpret_cast<uintptr_t>(src + size_t(feed) * NFP) & ~uintptr_t(127);
        const uintptr_t a = disc + uintptr_t(lane) * 128;
        if (a < end) discard_l2_line(reinterpret_cast<const void*>(a));
        const uintptr_t nd = disc + 32 * 128;
        disc = end > disc ? (end < nd ? end : nd) : disc;
      }
      wd.start();
      if (feed > rows && !L.first_slab && band == 0 && L.ack_prev) {
        __syncwarp();
        if (lane == 0) st_relaxed_sys_u32(L.ack_prev, L.epoch);   // predecessor slab may reuse this ring
      }
      if (syn_feed_ns(DS) && n < 32) __nanosleep(syn_feed_ns(DS));
    } else {
      if (wd.expired(L)) return false;
      if (syn_feed_ns(DS)) __nanosleep(syn_feed_ns(DS));
    }
  }
  return true;
}

// Idle warps appended to each CTA: they only join the band barriers.  With one compute warp +
// one feeder per CTA, consecutive CTAs of an SM place their compute warps on the same SM
// sub-partitions; a CTA of 2 + 2 warps moves the next CTA's compute warp to another one.
// Measured (interleaved A/B, one-warp variant): dsize 5 tsize 10 (C5b) 9.16 -> 8.60 ms,
// tsize 100 63.0 -> 61.6 ms, tsize 1000 (dim 4096) unchanged; dsize 1 tsize 10 (C5a) +0.6 %,
// tsize 1000 (C5c) +1.5 %, so only many-plane cells (dsize >= 3, the 16-row-window regime) get it.
// WF_SYN_PAD >= 0 forces the count (experiments).
#ifndef WF_SYN_PAD
#define WF_SYN_PAD -1
#endif
__host__ __device__ constexpr int syn_pad(int ds) { return WF_SYN_PAD >= 0 ? WF_SYN_PAD : (ds >= 3 ? 2 : 0); }
template <int DS, int K, int WARPS, int TS>
__global__ void __launch_bounds__((WARPS + 1 + syn_pad(DS)) * 32)
    syn_kernel(const SweepLaunch L, const PolSyn<DS> pol, const __grid_constant__ SynMaps maps) {
  using S = SynSmem<DS, K, WARPS>;
  extern __shared__ __align__(16) unsigned char syn_smem_raw[];
  const S sm(syn_smem_raw);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  for (int band = blockIdx.x; band < L.nbands; band += gridDim.x) {
    if (threadIdx.x < 64) sm.rprog[threadIdx.x] = 0;   // rprog and wprog
    __syncthreads();
    if (warp == WARPS) {
      syn_feeder<DS, K, WARPS>(L, pol, sm, band, lane);
    } else if (warp < WARPS) {
      SynWarp<DS, K, WARPS, TS> w(L, pol, maps, sm, band, warp, lane);
      w.run();
    }
    __syncthreads();
    if (run_failed(L)) return;
  }
}

// Plane-split kernel (impl 8): one 32-column band per CTA, DS compute warps (warp d computes
// float item d, warp 0 also the int fields) + the feeder (warp DS), which recycles a west-ring
// slot once every plane warp has consumed it.
template <int DS, int TS, int PW>
__device__ __forceinline__ void syn_ps_dispatch(const SweepLaunch& L, const PolSyn<DS>& pol, const SynMaps& maps,
                                                const SynSmem<DS, 1, 1>& sm, int band, int warp, int lane) {
  if constexpr (PW < DS) {
    if (warp == PW) {
      SynWarp<DS, 1, 1, TS, PW> w(L, pol, maps, sm, band, 0, lane);
      w.run();
    } else {
      syn_ps_dispatch<DS, TS, PW + 1>(L, pol, maps, sm, band, warp, lane);
    }
  }
}

template <int DS, int TS>
__global__ void __launch_bounds__((DS + 1) * 32)
    syn_ps_kernel(const SweepLaunch L, const PolSyn<DS> pol, const __grid_constant__ SynMaps maps) {
  using S = SynSmem<DS, 1, 1>;
  extern __shared__ __align__(16) unsigned char syn_smem_raw[];
  const S sm(syn_smem_raw);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  for (int band = blockIdx.x; band < L.nbands; band += gridDim.x) {
    if (threadIdx.x < 64) sm.rprog[threadIdx.x] = 0;   // rprog and wprog
    __syncthreads();
    if (warp == DS) syn_feeder<DS, 1, 1, DS>(L, pol, sm, band, lane);
    else syn_ps_dispatch<DS, TS, 0>(L, pol, maps, sm, band, warp, lane);
    __syncthreads();
    if (run_failed(L)) return;
  }
}

cudaError_t encode_plane_map_f(CUtensorMap* m, const SweepLaunch& L, int plane, int box_cols, int box_rows);

namespace {

template <int DS, int K, int W>
cudaError_t launch_syn(const SweepLaunch& L, cudaStream_t s, size_t smem) {
  PolSyn<DS> pol{};
  pol.u = static_cast<const float*>(L.row_in);
  pol.v = static_cast<const float*>(L.col_in);
  for (int d = 0; d < DS; ++d) {
    pol.topf[d] = static_cast<const float*>(L.top[d]);
    pol.leftf[d] = static_cast<const float*>(L.left[d]);
  }
  pol.tsize = L.tsize;
  SynMaps maps;
  memset(&maps, 0, sizeof maps);
  for (int f = 0; f < 2 + DS; ++f) {
    cudaError_t e = encode_plane_map_f(&maps.m[f], L, f, 32 * K, syn_ut(DS));
    if (e != cudaSuccess) return e;
  }
  // tsize of the BASELINE configs (10, 100, 1000) as a compile-time trip count for the
  // default one-column-per-lane variants of dsize 1 and 5
  auto kfn = syn_kernel<DS, K, W, 0>;
  if constexpr (K == 1 && (DS == 1 || DS == 5)) {
    if (L.tsize == 10) kfn = syn_kernel<DS, K, W, 10>;
    if (L.tsize == 100) kfn = syn_kernel<DS, K, W, 100>;
    if (L.tsize == 1000) kfn = syn_kernel<DS, K, W, 1000>;
  }
  cudaError_t e = cudaFuncSetAttribute(kfn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  kfn<<<L.grid, (W + 1 + syn_pad(DS)) * 32, smem, s>>>(L, pol, maps);
  return cudaGetLastError();
}

template <int DS>
cudaError_t launch_syn_ps(const SweepLaunch& L, cudaStream_t s, size_t smem) {
  PolSyn<DS> pol{};
  pol.u = static_cast<const float*>(L.row_in);
  pol.v = static_cast<const float*>(L.col_in);
  for (int d = 0; d < DS; ++d) {
    pol.topf[d] = static_cast<const float*>(L.top[d]);
    pol.leftf[d] = static_cast<const float*>(L.left[d]);
  }
  pol.tsize = L.tsize;
  SynMaps maps;
  memset(&maps, 0, sizeof maps);
  for (int f = 0; f < 2 + DS; ++f) {
    cudaError_t e = encode_plane_map_f(&maps.m[f], L, f, 32, syn_ut(DS));
    if (e != cudaSuccess) return e;
  }
  auto kfn = syn_ps_kernel<DS, 0>;
  if constexpr (DS == 5) {
    if (L.tsize == 100) kfn = syn_ps_kernel<DS, 100>;
    if (L.tsize == 1000) kfn = syn_ps_kernel<DS, 1000>;
  }
  cudaError_t e = cudaFuncSetAttribute(kfn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  kfn<<<L.grid, (DS + 1) * 32, smem, s>>>(L, pol, maps);
  return cudaGetLastError();
}

template <int DS>
Variant make_syn_ps() {
  using S = SynSmem<DS, 1, 1>;
  Variant v{WF_FN_SYNTHETIC, DS, 1, 1, 1, (DS + 1) * 32, S::bytes,
            reinterpret_cast<const void*>(syn_ps_kernel<DS, 0>), &launch_syn_ps<DS>, 8, {}};
  if constexpr (DS == 5) {
    v.alt[0] = reinterpret_cast<const void*>(syn_ps_kernel<DS, 100>);
    v.alt[1] = reinterpret_cast<const void*>(syn_ps_kernel<DS, 1000>);
  }
  return v;
}

template <int DS, int K, int W>
Variant make_syn() {
  using S = SynSmem<DS, K, W>;
  Variant v{WF_FN_SYNTHETIC, DS, K, W, 1, (W + 1 + syn_pad(DS)) * 32, S::bytes,
            reinterpret_cast<const void*>(syn_kernel<DS, K, W, 0>), &launch_syn<DS, K, W>, 7, {}};
  if constexpr (K == 1 && (DS == 1 || DS == 5)) {   // the compile-time tsize kernels launch_syn picks
    v.alt[0] = reinterpret_cast<const void*>(syn_kernel<DS, K, W, 10>);
    v.alt[1] = reinterpret_cast<const void*>(syn_kernel<DS, K, W, 100>);
    v.alt[2] = reinterpret_cast<const void*>(syn_kernel<DS, K, W, 1000>);
  }
  return v;
}

#define WF_SYN7(DS) make_syn<DS, 1, 1>(), make_syn<DS, 1, 2>(), make_syn<DS, 1, 4>(), make_syn<DS, 2, 2>()

}  // namespace

const Variant* syn_table(size_t* n) {
#ifdef WF_MIN_VARIANTS
  static const Variant v[] = {WF_SYN7(1), WF_SYN7(5), make_syn_ps<5>()};
#else
  static const Variant v[] = {WF_SYN7(0), WF_SYN7(1), WF_SYN7(2), WF_SYN7(3), WF_SYN7(4),
                              WF_SYN7(5), WF_SYN7(6), WF_SYN7(7), WF_SYN7(8),
                              make_syn_ps<2>(), make_syn_ps<3>(), make_syn_ps<4>(), make_syn_ps<5>(),
                              make_syn_ps<6>(), make_syn_ps<7>(), make_syn_ps<8>()};
#endif
  *n = sizeof(v) / sizeof(v[0]);
  return v;
}

}  // namespace wfk
