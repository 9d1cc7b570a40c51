// wf_nw.cuh -- the sequence-comparison (Needleman-Wunsch) band sweep, specialised for
// the B200 issue pipeline.  Same band / lane / skew model as
// wf_sweep.cuh (read that header first); what differs, each step measured (profiles/):
//
//  * Compute warps issue NO global memory operations in the row loop.  One I/O warp per
//    CTA (a) stages the row codes x_i into a shared x ring, (b) feeds the band's west
//    column (column-0 boundary, or the previous band's global LL ring) into a shared feed
//    ring for compute warp 0, and (c) forwards the last compute warp's east column to
//    the next band's / next slab's global LL ring.
//  * The row loop runs in blocks of U steps.  A warp's U finished rows sit in its staging
//    ring (shared memory, row-major, the TMA source).  After each block the warp executes
//    ONE fence (fence.proxy.async: MEMBAR.ALL.CTA + async-proxy view fence), after which
//    lane 0 both issues the block's TMA 2-D tensor store (UTMASTG) and publishes the
//    warp's progress counter.  The NEXT warp reads its west inputs -- the producer's east
//    column -- straight out of that staging ring: one shared load per 32-row block, no
//    per-row handoff traffic and no extra fence.
//  * Lane 0's west value and row code come from those per-block loads by indexed
//    shuffle; every other lane receives both from its left neighbour by __shfl_up_sync
//    (the row codes travel with the lane skew).
//  * Ramp-up and drain blocks carry a per-lane "row in range" predicate; steady blocks do
//    not.  The tensor bounds clip drain rows > rows and the ragged last band.
//  * The cell, with W entering last (R9), in prefix form:
//        s   = score(x_i, y_j)                  PRMT byte lookup (alphabet <= 8) or ISETP+SEL
//        t1  = max(N + g, NW + s)               IADD + VIADDMNMX
//        P_m = max(t1_m, P_{m-1} + g)           VIADDMNMX (depends on the previous row only)
//        H_m = max(P_m, W + (m+1) g)            VIADDMNMX: W reaches every cell in ONE op
//    which is the same integer as max(t1_m, H_{m-1} + g) unrolled along the lane's row.
#pragma once
#include <cuda.h>

#include "wf_cells.cuh"
#include "wf_sweep.cuh"

namespace wfk {

constexpr int kXRing = 4096;   // rows of x codes staged ahead in shared memory (power of 2)
constexpr int kFeed = 256;     // rows in the I/O warp's west-feed ring (power of 2)

template <int D, int U>
__host__ __device__ constexpr int nw_ring_rows() {
  // rows pending in a warp's staging ring: 31D (lane skew) + 2U (this block + the one the
  // next warp is still reading) + one block of TMA in flight
  return (31 * D + 3 * U) <= 64 ? 64 : (31 * D + 3 * U) <= 128 ? 128 : 256;
}

template <int K, int WARPS, int D, int U>
struct NwSmem {
  static constexpr int R = nw_ring_rows<D, U>();
  static constexpr int ROWB = 32 * K * 4;                                  // bytes per staged row
  static constexpr size_t stage_bytes = size_t(WARPS) * R * ROWB;
  static constexpr size_t feed_bytes = size_t(kFeed) * 4;
  static constexpr size_t ctl_bytes = 64 * 4;
  static constexpr size_t bytes = 1024 + stage_bytes + feed_bytes + kXRing + ctl_bytes;
  unsigned char* stage;     // [WARPS][R][32K] int32, 1024-byte aligned (TMA source rows)
  int32_t* feed;            // [kFeed] west column of warp 0, row r at r & (kFeed-1)
  unsigned char* xring;     // [kXRing] row codes, x of row r at (r-1) & (kXRing-1)
  int* wprog;               // wprog[w]: rows 1..wprog[w] of warp w's staging ring are published
                            //           (w = WARPS: the feed ring)
  int* rprog;               // rprog[w]: rows of warp w's staging ring / feed consumed by its reader
  int* xfill;               // rows 1..*xfill of the x ring are valid
  int* xneed;               // xneed[w]: lowest row warp w may still read from the x ring
  __device__ __forceinline__ explicit NwSmem(unsigned char* raw) {
    const uint32_t a = static_cast<uint32_t>(__cvta_generic_to_shared(raw));
    unsigned char* base = raw + ((1024u - (a & 1023u)) & 1023u);
    stage = base;
    feed = reinterpret_cast<int32_t*>(base + stage_bytes);
    xring = base + stage_bytes + feed_bytes;
    int* ctl = reinterpret_cast<int*>(xring + kXRing);
    wprog = ctl;          // [0..16)
    rprog = ctl + 16;     // [16..32)
    xneed = ctl + 32;     // [32..48)
    xfill = ctl + 48;
  }
};

__device__ __forceinline__ int32_t prmt_s8(uint32_t lo, uint32_t hi, uint32_t sel) {
  uint32_t r;
  asm("prmt.b32 %0, %1, %2, %3;" : "=r"(r) : "r"(lo), "r"(hi), "r"(sel));
  return static_cast<int32_t>(r);
}
__device__ __forceinline__ void fence_proxy_async_smem() { asm volatile("fence.proxy.async.shared::cta;" ::: "memory"); }
__device__ __forceinline__ void tma_store_2d(const CUtensorMap* map, uint32_t smem, int c, int r) {
  asm volatile("cp.async.bulk.tensor.2d.global.shared::cta.bulk_group [%0, {%1, %2}], [%3];" ::"l"(map), "r"(c),
               "r"(r), "r"(smem)
               : "memory");
}
__device__ __forceinline__ void bulk_commit() { asm volatile("cp.async.bulk.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void bulk_wait_read() {
  asm volatile("cp.async.bulk.wait_group.read %0;" ::"n"(N) : "memory");
}
__device__ __forceinline__ void bulk_wait_all() { asm volatile("cp.async.bulk.wait_group 0;" ::: "memory"); }
__device__ __forceinline__ int32_t lds_vol_s32(const void* p) {
  int32_t v;
  asm volatile("ld.volatile.shared.s32 %0, [%1];" : "=r"(v) : "r"(static_cast<uint32_t>(__cvta_generic_to_shared(p))));
  return v;
}
// Distributed shared memory (thread-block clusters): the address of the same shared
// variable in CTA `rank` of this cluster, and relaxed / release accesses to it.
__device__ __forceinline__ uint32_t dsmem_addr(const void* local, uint32_t rank) {
  uint32_t r;
  asm volatile("mapa.shared::cluster.u32 %0, %1, %2;"
               : "=r"(r)
               : "r"(static_cast<uint32_t>(__cvta_generic_to_shared(local))), "r"(rank));
  return r;
}
__device__ __forceinline__ void st_cluster_u32(uint32_t a, uint32_t v) {
  asm volatile("st.relaxed.cluster.shared::cluster.u32 [%0], %1;" ::"r"(a), "r"(v) : "memory");
}
__device__ __forceinline__ void st_release_cluster_u32(uint32_t a, uint32_t v) {
  asm volatile("st.release.cluster.shared::cluster.u32 [%0], %1;" ::"r"(a), "r"(v) : "memory");
}
__device__ __forceinline__ uint32_t ld_cluster_u32(uint32_t a) {
  uint32_t v;
  asm volatile("ld.relaxed.cluster.shared::cluster.u32 %0, [%1];" : "=r"(v) : "r"(a) : "memory");
  return v;
}
__device__ __forceinline__ void fence_acq_rel_cluster() { asm volatile("fence.acq_rel.cluster;" ::: "memory"); }
__device__ __forceinline__ void cluster_sync_all() {
  asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
}
__device__ __forceinline__ uint32_t cluster_ctarank() {
  uint32_t r;
  asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
  return r;
}
constexpr int kClusterSize = 8;   // largest (portable) cluster size; L.cluster holds the launched size

__device__ __forceinline__ uint32_t lds_u8(const unsigned char* p) {
  uint32_t v;
  asm volatile("ld.volatile.shared.u8 %0, [%1];" : "=r"(v) : "r"(static_cast<uint32_t>(__cvta_generic_to_shared(p))));
  return v;
}

// =====================================================================================
// Compute warp: lane l owns K adjacent columns; at step t it is on row t - D*l + 1.
// =====================================================================================
// LOCAL = Smith-Waterman (R9): H = max(0, NW + s, N + g, W + g),
// boundary 0.  The floor rides on the same VIADDMNMX (its .RELU form), so
// max(t1_m, H_{m-1} + g) and the prefix form stay exact; the lane also tracks its best cell
// value and the first row reaching it (the fused best-cell reduction, finished by
// sw_best_kernel in wf_sw.cu).
template <int K, int WARPS, int D, int U, bool PRMT, bool LOCAL = false, bool CL = false>
struct NwWarp {
  using S = NwSmem<K, WARPS, D, U>;
  static constexpr int R = S::R;
  static constexpr int ROWB = S::ROWB;
  static_assert(U == 32 || U == 16, "block height");
  static_assert(R % U == 0 && kFeed % U == 0, "block alignment");
#ifndef WF_NW_PREFIX
#define WF_NW_PREFIX 1
#endif
  static constexpr bool kPrefix = WF_NW_PREFIX != 0;

  const SweepLaunch& L;
  const CUtensorMap* tmap;
  const S& sm;
  const int band, warp, lane;
  int rows;
  int32_t gap, mmatch, mmis;
  int32_t gk[K];             // (m+1)*gap (prefix form)
  uint32_t qlo[K], qhi[K];   // PRMT: byte c = score(c, y_j) (int8) for c = 0..7
  uint32_t ycode[K];         // compare/select path
  int32_t Np[K];             // previous row at the lane's K columns
  int32_t prevW;             // previous row's west input (NW of the first column)
  int32_t q[D];              // east values of lane-1; q[D-1] is this step's west input
  uint32_t xq[D];            // row codes travelling with q
  int wcol;                  // warp's first column, slab-relative
  unsigned char* stage_w;    // this warp's staging ring
  unsigned char* stage_lane; // + lane's segment
  // west source: warp 0 reads the feed ring (stride 4 B), warp w > 0 the east column of
  // warp w-1's staging ring (stride ROWB)
  const unsigned char* wsrc;
  int wstride, wmask, wsrc_off;
  // Block phase and staging-ring row offset.  Warp w runs blocks starting at steps
  // t0 == -1 - 31*D*w (mod U), so its lane 0's rows t0+1 .. t0+U are exactly one block
  // published by warp w-1 (whose lane-31 rows lag its lane-0 rows by 31*D).  Row r lives in
  // ring slot (r + ring_off) & (R-1) with ring_off = 31*D*(w+1) mod U, which makes every
  // published block (rows r31_0 .. r31_0+U-1) contiguous for the TMA box.
  int phase, ring_off;
  int seen_wprog, seen_rprog, seen_xfill;
  int32_t best = 0;          // LOCAL: the lane's best cell value so far (cells are >= 0) ...
  int32_t best_row = 0;      // ... and the first row reaching it (0: none above 0 yet)
  __device__ __forceinline__ static int32_t t1f(int32_t N, int32_t g, int32_t d) {
    if constexpr (LOCAL) return __viaddmax_s32_relu(N, g, d);   // max(N + g, d, 0)
    else return __viaddmax_s32(N, g, d);
  }
  Watchdog wd;

  __device__ __forceinline__ NwWarp(const SweepLaunch& L_, const CUtensorMap* tmap_, const S& sm_, int band_,
                                    int warp_, int lane_)
      : L(L_), tmap(tmap_), sm(sm_), band(band_), warp(warp_), lane(lane_) {
    rows = L.rows;
    gap = L.gap;
    mmatch = L.match;
    mmis = L.mismatch;
#ifndef WF_NW_OPAQUE_GK
#define WF_NW_OPAQUE_GK 0
#endif
#pragma unroll
    for (int m = 0; m < K; ++m) {
      gk[m] = (m + 1) * gap;
      if (WF_NW_OPAQUE_GK) asm volatile("mov.b32 %0, %0;" : "+r"(gk[m]));   // keep W + gk[m] a DPX add-max
    }
    const uint8_t* y = static_cast<const uint8_t*>(L.col_in);
    wcol = band * L.band_w + warp * 32 * K;
    const int jb = L.c0 + wcol + lane * K;    // global 0-based column of the lane's first column
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
      Np[m] = (vc && !LOCAL) ? (jb + m + 1) * gap : 0;   // H[0][j] = j*g (NW), 0 (SW)
    }
    prevW = (jb < L.c1 && !LOCAL) ? jb * gap : 0;          // H[0][jb]
#pragma unroll
    for (int d = 0; d < D; ++d) {
      q[d] = 0;
      xq[d] = 0;
    }
    stage_w = sm.stage + size_t(warp) * R * ROWB;
    stage_lane = stage_w + lane * (4 * K);
    // phases follow the GLOBAL warp index (bands of all slabs form one chain)
#ifndef WF_NW_GLOBAL_PHASE
#define WF_NW_GLOBAL_PHASE 0
#endif
    const int gw = WF_NW_GLOBAL_PHASE ? (L.c0 / L.band_w + band) * WARPS + warp : warp;
    phase = ring_phase(gw);
    ring_off = ring_offset(gw);
    if (warp == 0) {
      wsrc = reinterpret_cast<const unsigned char*>(sm.feed);
      wstride = 4;
      wmask = kFeed - 1;
      wsrc_off = 0;
    } else {
      wsrc = sm.stage + size_t(warp - 1) * R * ROWB + (32 * K - 1) * 4;
      wstride = ROWB;
      wmask = R - 1;
      wsrc_off = ring_offset(gw - 1);
    }
    seen_wprog = seen_rprog = seen_xfill = 0;
  }

  static __host__ __device__ __forceinline__ int ring_phase(int w) { return ((-1 - 31 * D * w) % U + U) % U; }
  static __host__ __device__ __forceinline__ int ring_offset(int w) { return (31 * D * (w + 1)) % U; }

  __device__ __forceinline__ void cells(int32_t Win, uint32_t xc, int32_t (&H)[K]) const {
    const uint32_t sel = xc * 0x1111u + 0x8880u;   // byte xc, sign-replicated (prmt default mode)
    if constexpr (kPrefix) {
      int32_t P = 0;
#pragma unroll
      for (int m = 0; m < K; ++m) {
        const int32_t NW = m == 0 ? prevW : Np[m - 1];
        int32_t s;
        if constexpr (PRMT) s = prmt_s8(qlo[m], qhi[m], sel);
        else s = (xc == ycode[m]) ? mmatch : mmis;
        const int32_t t1 = t1f(Np[m], gap, NW + s);
        P = (m == 0) ? t1 : __viaddmax_s32(P, gap, t1);
        H[m] = __viaddmax_s32(Win, gk[m], P);
      }
    } else {
#pragma unroll
      for (int m = 0; m < K; ++m) {
        const int32_t NW = m == 0 ? prevW : Np[m - 1];
        const int32_t W = m == 0 ? Win : H[m - 1];
        int32_t s;
        if constexpr (PRMT) s = prmt_s8(qlo[m], qhi[m], sel);
        else s = (xc == ycode[m]) ? mmatch : mmis;
        const int32_t t1 = t1f(Np[m], gap, NW + s);
        H[m] = __viaddmax_s32(W, gap, t1);
      }
    }
  }

  __device__ __forceinline__ void stage_store(int row, const int32_t (&H)[K]) const {
    unsigned char* dst = stage_lane + ((row + ring_off) & (R - 1)) * ROWB;
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

  // plain copy of the finished row r from the staging ring to HBM (first block only: a
  // negative start row is not a legal TMA store coordinate)
  __device__ __forceinline__ void write_row(int r) const {
    const int jrel = wcol + lane * K;
    const int width = L.c1 - L.c0;
    const uint32_t* src = reinterpret_cast<const uint32_t*>(stage_lane + ((r + ring_off) & (R - 1)) * ROWB);
    uint32_t* dst = static_cast<uint32_t*>(L.out[0]) + int64_t(r - 1) * L.pitch + jrel;
#pragma unroll
    for (int m = 0; m < K; ++m)
      if (jrel + m < width) dst[m] = src[m];
  }

  // wait until a shared counter reaches `need` (uniform spin; `seen` caches the last value)
  __device__ __forceinline__ bool wait_ctr(const int* ctr, int need, int& seen, unsigned sleep_ns) {
    if (seen >= need) return true;
    wd.start();
    for (;;) {
      if constexpr (CL) {   // acquire at cluster scope: the feed counter may be released by the previous CTA
        uint32_t v;
        asm volatile("ld.acquire.cluster.shared::cta.u32 %0, [%1];"
                     : "=r"(v)
                     : "r"(static_cast<uint32_t>(__cvta_generic_to_shared(ctr)))
                     : "memory");
        seen = static_cast<int>(v);
        if (seen >= need) return true;
      } else {
        seen = lds_vol_i(ctr);
      }
      if (seen >= need) {
        // order the data reads after the observed counter (cluster scope: the feed ring may be
        // written by the previous band's CTA through DSMEM)
        if constexpr (CL) fence_acq_rel_cluster();
        else __threadfence_block();
        return true;
      }
      if (wd.expired(L)) return false;
#ifndef WF_NW_WAIT_SLEEP
#define WF_NW_WAIT_SLEEP 1     // 0: compute warps spin on shared counters without back-off
#endif
      if (WF_NW_WAIT_SLEEP) __nanosleep(sleep_ns);
    }
  }

#ifndef WF_NW_ROT
#define WF_NW_ROT 0
#endif
  // Rotation form (D = 1): lane 31 hands lane 0 its next west input and row code through the
  // same lane-rotating shuffle that carries every other lane's east value, so the only
  // instructions on the lane-to-lane chain are SHFL and one VIADDMNMX:
  //   src = max(W + gL, PL), gL = K*g, PL = P_{K-1} (lanes 0..30)  -> H[K-1]
  //                          gL = -2^28, PL = w0 of the next row (lane 31) -> w0'
  template <bool EDGE>
  __device__ __forceinline__ void block_rot(int t0, int32_t wv, uint32_t xv, int32_t& east_last) {
    const int src_lane = (lane + 31) & 31;
    int32_t gL;
    asm volatile("mov.b32 %0, %1;" : "=r"(gL) : "r"(lane == 31 ? -(1 << 28) : K * gap));
    const int32_t w00 = __shfl_sync(0xffffffffu, wv, 0);    // shuffles outside the selects:
    const uint32_t x00 = __shfl_sync(0xffffffffu, xv, 0);   // every lane must execute them
    int32_t Win = (lane == 0) ? w00 : q[0];
    uint32_t Xin = (lane == 0) ? x00 : xq[0];
#pragma unroll
    for (int u = 0; u < U; ++u) {
      const int row = t0 + u - lane + 1;
      const int32_t w0n = __shfl_sync(0xffffffffu, wv, (u + 1) & (U - 1));   // next row of lane 0
      const uint32_t x0n = __shfl_sync(0xffffffffu, xv, (u + 1) & (U - 1));
      int32_t H[K];
      int32_t Pl;
      cells_p(Win, Xin, H, Pl);
      const int32_t PL = (lane == 31) ? w0n : Pl;
      const int32_t src = __viaddmax_s32(Win, gL, PL);
      const uint32_t xsrc = (lane == 31) ? x0n : Xin;
      if constexpr (EDGE) {
        const bool active = row >= 1 && row <= rows;
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
      Win = __shfl_sync(0xffffffffu, src, src_lane);
      Xin = __shfl_sync(0xffffffffu, xsrc, src_lane);
    }
    // lanes 1..31 carry their next west input into the next block in q[0]
    q[0] = Win;
    xq[0] = Xin;
    east_last = Np[K - 1];
  }

  // prefix cells returning P_{K-1} as well (the rotation form recomputes H[K-1] for lane 31)
  __device__ __forceinline__ void cells_p(int32_t Win, uint32_t xc, int32_t (&H)[K], int32_t& Plast) const {
    const uint32_t sel = xc * 0x1111u + 0x8880u;
    int32_t P = 0;
#pragma unroll
    for (int m = 0; m < K; ++m) {
      const int32_t NW = m == 0 ? prevW : Np[m - 1];
      int32_t s;
      if constexpr (PRMT) s = prmt_s8(qlo[m], qhi[m], sel);
      else s = (xc == ycode[m]) ? mmatch : mmis;
      const int32_t t1 = t1f(Np[m], gap, NW + s);
      P = (m == 0) ? t1 : __viaddmax_s32(P, gap, t1);
      H[m] = __viaddmax_s32(Win, gk[m], P);
    }
    Plast = P;
  }

  template <bool EDGE>
  __device__ __forceinline__ void block(int t0, int32_t wv, uint32_t xv, int32_t& east_last) {
    if constexpr (WF_NW_ROT != 0 && D == 1) {
      block_rot<EDGE>(t0, wv, xv, east_last);
      return;
    }
#pragma unroll
    for (int u = 0; u < U; ++u) {
      const int row = t0 + u - D * lane + 1;
      const int32_t w0 = __shfl_sync(0xffffffffu, wv, u);        // lane 0: west input of row t0+u+1
      const uint32_t x0 = __shfl_sync(0xffffffffu, xv, u);       // lane 0: its row code
      const int32_t Win = (lane == 0) ? w0 : q[D - 1];
      const uint32_t Xin = (lane == 0) ? x0 : xq[D - 1];
      int32_t H[K];
      cells(Win, Xin, H);
      if constexpr (LOCAL) {   // best cell: strict > keeps the first row reaching the value
        int32_t rm = H[0];
#pragma unroll
        for (int m = 1; m < K; ++m) rm = max(rm, H[m]);
        const bool up = rm > best && (!EDGE || (row >= 1 && row <= rows));
        best = up ? rm : best;
        best_row = up ? row : best_row;
      }
      if constexpr (EDGE) {   // ramp-up / drain: predicated selects, no divergent branch
        const bool active = row >= 1 && row <= rows;
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
      const int32_t r = __shfl_up_sync(0xffffffffu, Np[K - 1], 1);
      const uint32_t rx = __shfl_up_sync(0xffffffffu, Xin, 1);
#pragma unroll
      for (int d = D - 1; d > 0; --d) {
        q[d] = q[d - 1];
        xq[d] = xq[d - 1];
      }
      q[0] = r;
      xq[0] = rx;
    }
    east_last = Np[K - 1];
  }

  __device__ __forceinline__ bool run() {
    const int T = rows + 31 * D;                  // steps
    int t0 = phase - U;                           // first block start (<= -1), t0 == phase (mod U)
    const int steady_lo = 31 * D;                 // t >= 31D: lane 31's row >= 1
    const int steady_hi = rows - U;               // t0 + U - 1 <= rows - 1: lane 0's row <= rows
    const int* wprog_src = sm.wprog + (warp == 0 ? WARPS : warp - 1);
    int* rprog_src = sm.rprog + (warp == 0 ? WARPS : warp - 1);
    const uint32_t stage_w_s = static_cast<uint32_t>(__cvta_generic_to_shared(stage_w));
    if (L.trace && warp == 0 && lane == 0) {
      L.trace[size_t(band) * kTraceSlots] = globaltimer();
      L.trace[size_t(band) * kTraceSlots + 42] = clock64();
    }
    int blk = 0;
    // WF_TRACE phase profile (lane 0 of warps 0..2): SM cycles spent per block phase --
    // [0] west wait, [1] west loads, [2] free-slot wait, [3] row compute, [4] publish
    const bool prof = L.trace != nullptr && lane == 0 && warp < 3;
    long long ph[5] = {0, 0, 0, 0, 0};
    long long tc = prof ? clock64() : 0;
    auto tick = [&](int i) {
      if (prof) {
        const long long n = clock64();
        ph[i] += n - tc;
        tc = n;
      }
    };
    // Instruction-cache warm-up (WF_NW_WARM): the steady and edge block bodies are ~100 KB of
    // unrolled SASS, and every band's first pass through them was paying the misses on the
    // band-to-band critical path.  A band that waits for its west input anyway first runs one
    // steady and one edge block through the SAME call site on dummy inputs (their staging
    // stores land in slots that real rows overwrite before any publish), then restores the
    // lane state.  Band 0 of the first slab starts at once and skips it.
#ifndef WF_NW_WARM
#define WF_NW_WARM 1
#endif
    int warm = (WF_NW_WARM && !(L.first_slab && band == 0)) ? 2 : 0;
    int32_t sv_Np[K], sv_q[D];
    uint32_t sv_xq[D];
    const int32_t sv_prevW = prevW, sv_best = best, sv_best_row = best_row;
#pragma unroll
    for (int m = 0; m < K; ++m) sv_Np[m] = Np[m];
#pragma unroll
    for (int d = 0; d < D; ++d) {
      sv_q[d] = q[d];
      sv_xq[d] = xq[d];
    }
    for (; t0 < T;) {
      const int r0 = t0 + 1;                       // lane 0's first row in this block
      const int rl = min(t0 + U, rows);            // its last valid row
      // ---- west inputs and row codes of lane 0's rows r0 .. r0+U-1: one shared load each
      int32_t wv = 0;
      uint32_t xv = 0;
      if (!warm && rl >= 1) {
        if (!wait_ctr(wprog_src, rl, seen_wprog, 20)) return false;
        if (!wait_ctr(sm.xfill, rl, seen_xfill, 32)) return false;
        tick(0);
        const int r = r0 + lane;
        if (lane < U && r >= 1 && r <= rows) {
          wv = lds_vol_s32(wsrc + ((r + wsrc_off) & wmask) * wstride);
          xv = lds_u8(sm.xring + ((r - 1) & (kXRing - 1)));
        }
      }
      // rows < r0 of the source are no longer needed (the loads above are complete once
      // used; publish one block late to be safe)
      if (!warm && lane == 0 && blk > 0) {
        sts_vol_i(rprog_src, r0 - U - 1 + U);
        sts_vol_i(sm.xneed + warp, r0);
      }
      tick(1);
      // ---- my staging ring: slots of rows <= lane 0's rows of this block minus R must be
      //      free: read by TMA (bulk groups) and by my reader (rprog[warp])
      const int need_free = t0 + U - R;
      if (!warm && need_free >= 1) {
        if (lane == 0) bulk_wait_read<1>();
        __syncwarp();
        if (!wait_ctr(sm.rprog + warp, need_free, seen_rprog, 20)) return false;
      }
      tick(2);
      int32_t east_last;
      if (!warm && L.trace && lane == 0 && t0 <= steady_lo && t0 + U > steady_lo)   // entering steady state
        L.trace[size_t(band) * kTraceSlots + 33 + warp] = globaltimer();
      const int tb = warm == 2 ? steady_lo : warm == 1 ? -4 * U : t0;   // block start step
      if (tb >= steady_lo && tb <= steady_hi) block<false>(tb, wv, xv, east_last);
      else block<true>(tb, wv, xv, east_last);
      (void)east_last;
      if (warm) {
        if (--warm == 0) {   // restore the lane state the dummy blocks advanced
          prevW = sv_prevW;
          best = sv_best;
          best_row = sv_best_row;
#pragma unroll
          for (int m = 0; m < K; ++m) Np[m] = sv_Np[m];
#pragma unroll
          for (int d = 0; d < D; ++d) {
            q[d] = sv_q[d];
            xq[d] = sv_xq[d];
          }
        }
        continue;
      }
      tick(3);
      wf_jitter(13);
      // ---- publish: one fence for the TMA engine and for the next warp
      const int r31_0 = t0 - 31 * D + 1;           // first row of the block's TMA box
      const int r31_last = min(r31_0 + U - 1, rows);
      if (r31_last >= 1) {
        fence_proxy_async_smem();
        __syncwarp();
        if (r31_0 >= 1) {
          if (lane == 0) {
            tma_store_2d(tmap, stage_w_s + ((r31_0 + ring_off) & (R - 1)) * ROWB, wcol, r31_0 - 1);
            bulk_commit();
          }
        } else {
#ifndef WF_NW_EARLY_PUB
#define WF_NW_EARLY_PUB 1
#endif
          // first block: publish before the generic-store write-back (the reader only needs the
          // staging ring, fenced above, and these slots are not reused before row R), so the
          // next warp's start does not wait for 32 rows of STGs
          if (WF_NW_EARLY_PUB && lane == 0) sts_vol_i(sm.wprog + warp, r31_last);
          for (int r = 1; r <= r31_last; ++r) write_row(r);
        }
        if (lane == 0) sts_vol_i(sm.wprog + warp, r31_last);
      }
      tick(4);
#ifdef WF_NW_TRACE_BLOCKS   // ramp cadence: end of the first 15 blocks (perturbs the code layout)
      if (L.trace && lane == 0 && warp < 2 && blk < 15)
        L.trace[size_t(band) * kTraceSlots + 1 + 15 * warp + blk] = globaltimer();
#endif
      t0 += U;
      ++blk;
    }
    if (prof)
      for (int i = 0; i < 5; ++i) L.trace[size_t(band) * kTraceSlots + 48 + 5 * warp + i] = ph[i];
    if (lane == 0) {
      bulk_wait_all();
      sts_vol_i(rprog_src, rows);
      sts_vol_i(sm.xneed + warp, rows + 1);
    }
    if (L.trace && warp == 0 && lane == 0) {
      L.trace[size_t(band) * kTraceSlots + kTraceRows] = globaltimer();
      L.trace[size_t(band) * kTraceSlots + 43] = clock64();
    }
    if constexpr (LOCAL) L.lane_best[(size_t(band) * WARPS + warp) * 32 + lane] = make_int2(best, best_row);
    return true;
  }
};

// =====================================================================================
// I/O warp: x staging, west feed of warp 0, east forwarding of warp WARPS-1.
// =====================================================================================
template <int K, int WARPS, int D, int U, bool LOCAL = false, bool CL = false>
__device__ __forceinline__ bool nw_io_warp(const SweepLaunch& L, const NwSmem<K, WARPS, D, U>& sm, int band,
                                           int lane) {
  using S = NwSmem<K, WARPS, D, U>;
  const int rows = L.rows;
  const uint8_t* x = static_cast<const uint8_t*>(L.row_in);
  const bool boundary = L.first_slab && band == 0;
  const unsigned long long* src = L.edge + size_t(band) * edge_stride(rows);                 // inbound ring
  unsigned long long* dst = (band + 1 < L.nbands) ? L.edge + size_t(band + 1) * edge_stride(rows) : L.next_edge;
  const bool wait_ack = band + 1 >= L.nbands && L.next_edge && L.ack_self;
  const unsigned char* east_col = sm.stage + size_t(WARPS - 1) * S::R * S::ROWB + (32 * K - 1) * 4;
  const int last_off = NwWarp<K, WARPS, D, U, true>::ring_offset(
      WF_NW_GLOBAL_PHASE ? (L.c0 / L.band_w + band) * WARPS + WARPS - 1 : WARPS - 1);
  // Cluster mode: the previous band of this round runs in the CTA of cluster rank - 1 and
  // writes this CTA's feed ring itself (DSMEM); this band's east column goes to rank + 1.
  const uint32_t crank = CL ? cluster_ctarank() : 0u;
  const bool from_cluster = CL && crank > 0 && band > 0;
  const bool to_cluster = CL && crank + 1 < static_cast<uint32_t>(L.cluster) && band + 1 < L.nbands &&
                          blockIdx.x + 1 < gridDim.x;
  uint32_t r_feed = 0, r_wprog = 0, r_rprog = 0;
  if (to_cluster) {
    r_feed = dsmem_addr(sm.feed, crank + 1);
    r_wprog = dsmem_addr(sm.wprog + WARPS, crank + 1);
    r_rprog = dsmem_addr(sm.rprog + WARPS, crank + 1);
  }
  // I/O warp back-off (ns) after a productive / idle pass.  With WARPS <= 2 the I/O warp
  // (warp WARPS) has an SM sub-partition of its own, so it spins without sleeping: measured
  // C4 2.718 -> 2.659 ms (profiles/r01_io_spin_ab.txt).  Otherwise it shares a scheduler with
  // compute warp 0 and backs off.
#ifndef WF_NW_IO_NS_BUSY
#define WF_NW_IO_NS_BUSY (WARPS <= 2 ? 0 : 64)
#endif
#ifndef WF_NW_IO_NS_IDLE
#define WF_NW_IO_NS_IDLE (WARPS <= 2 ? 0 : 128)
#endif
#ifndef WF_NW_LL_GPU
#define WF_NW_LL_GPU 0         // 1: band-to-band rings on this device use .gpu-scope LL accesses
#endif
  // the inbound ring is written by this device unless it is band 0 of a slab g > 0 (peer GPU)
  const bool src_local = WF_NW_LL_GPU && band > 0;
  const bool dst_local = WF_NW_LL_GPU && band + 1 < L.nbands;
  int feed = from_cluster ? rows + 1 : 1;   // next row to feed (the producer feeds a cluster band)
  int fwd = 1;                  // next row to forward from the last warp's staging ring
  int seen_feed_rd = 0, seen_last_wr = 0, seen_remote_rd = 0;
  bool acked = !wait_ack;
  Watchdog wd;
  wd.start();
  while (feed <= rows || fwd <= rows) {
    wf_jitter(11);
    bool progress = false;
    // (b) west feed of compute warp 0 (boundary column or the previous band's LL ring)
    if (feed <= rows) {
      const int need = feed + 63 - kFeed;    // slot reuse: warp 0 has consumed those rows
      if (seen_feed_rd < need) seen_feed_rd = lds_vol_i(sm.rprog + WARPS);
      if (seen_feed_rd >= need) {
        int32_t v[2];
        bool ok[2];
#pragma unroll
        for (int h = 0; h < 2; ++h) {
          const int r = feed + h * 32 + lane;
          ok[h] = true;
          v[h] = 0;
          if (r <= rows) {
            if (boundary) {
              v[h] = LOCAL ? 0 : r * L.gap;                       // H[r][0] = r*g (NW), 0 (SW)
            } else {
              const unsigned long long wv = src_local ? ld_relaxed_gpu(src + r) : ld_relaxed_sys(src + r);
              v[h] = static_cast<int32_t>(static_cast<uint32_t>(wv));
              ok[h] = static_cast<uint32_t>(wv >> 32) == L.epoch;
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
            if (r < feed + n) sm.feed[r & (kFeed - 1)] = v[h];
          }
          __syncwarp();
          __threadfence_block();
          feed += n;
          if (lane == 0) sts_vol_i(sm.wprog + WARPS, feed - 1);
          if (L.trace && lane == 0 && feed - n <= 32 && feed > 32)   // first 32 rows fed
            L.trace[size_t(band) * kTraceSlots + 37] = globaltimer();
          progress = true;
          if (feed > rows && !L.first_slab && band == 0 && L.ack_prev && lane == 0)
            st_relaxed_sys_u32(L.ack_prev, L.epoch);   // predecessor slab may reuse this ring
        }
      }
    }
    // (c) forward the band's east column from the last warp's staging ring
    if (fwd <= rows) {
      if (!acked) {   // the next slab must have drained its ring in the previous run
        const unsigned a = ld_relaxed_sys_u32(L.ack_self);
        acked = static_cast<int>(a - (L.epoch - 1u)) >= 0;
      }
      if (acked) {
        if (seen_last_wr < fwd) {
          seen_last_wr = lds_vol_i(sm.wprog + WARPS - 1);
          if (seen_last_wr >= fwd) __threadfence_block();
        }
        int avail = min(seen_last_wr, rows) - fwd + 1;
        if (to_cluster && avail > 0) {   // the consumer's feed-ring slots must be free
          const int need = fwd + min(avail, 32) - 1 - kFeed;
          if (seen_remote_rd < need) seen_remote_rd = static_cast<int>(ld_cluster_u32(r_rprog));
          if (seen_remote_rd < need) avail = 0;
        }
        if (avail > 0) {
          const int n = min(avail, 32);
          const int r = fwd + lane;
          if (lane < n) {
            const int32_t v = lds_vol_s32(east_col + ((r + last_off) & (S::R - 1)) * S::ROWB);
            if (to_cluster) st_cluster_u32(r_feed + 4u * (r & (kFeed - 1)), static_cast<uint32_t>(v));
            else if (dst_local) st_relaxed_gpu(dst + r, ll_pack(static_cast<uint32_t>(v), L.epoch));
            else if (dst) st_relaxed_sys(dst + r, ll_pack(static_cast<uint32_t>(v), L.epoch));
          }
          __syncwarp();   // orders every lane's DSMEM store before lane 0's release of the counter
          if (to_cluster && lane == 0) st_release_cluster_u32(r_wprog, static_cast<uint32_t>(fwd + n - 1));
          fwd += n;
          if (lane == 0) sts_vol_i(sm.rprog + WARPS - 1, fwd - 1);
          if (L.trace && lane == 0 && fwd - n <= 32 && fwd > 32)     // first 32 rows forwarded
            L.trace[size_t(band) * kTraceSlots + 36] = globaltimer();
          progress = true;
        }
      }
    }
    if (progress) {
      wd.start();
      if (WF_NW_IO_NS_BUSY) __nanosleep(WF_NW_IO_NS_BUSY);
    } else {
      if (wd.expired(L)) return false;
      if (WF_NW_IO_NS_IDLE) __nanosleep(WF_NW_IO_NS_IDLE);
    }
  }
  return true;
}

// x-staging warp: keeps the shared x ring up to kXRing rows ahead of the slowest compute
// warp (a separate warp, so its global-load latency never delays the feed / forward duties)
template <int K, int WARPS, int D, int U>
__device__ __forceinline__ bool nw_x_warp(const SweepLaunch& L, const NwSmem<K, WARPS, D, U>& sm, int lane) {
  const int rows = L.rows;
  const uint8_t* x = static_cast<const uint8_t*>(L.row_in);
  int xfill = 0;
  Watchdog wd;
  wd.start();
  while (xfill < rows) {
    wf_jitter(12);
    int lo = rows + 1;
#pragma unroll
    for (int w = 0; w < WARPS; ++w) lo = min(lo, lds_vol_i(sm.xneed + w));
    const int cap = min(rows, lo - 1 + kXRing);
    if (cap > xfill) {
      const int n = min(cap - xfill, 1024);
      for (int i = lane; i < n; i += 32) {
        const int r = xfill + 1 + i;
        sm.xring[(r - 1) & (kXRing - 1)] = __ldg(x + (r - 1));
      }
      __syncwarp();
      __threadfence_block();
      xfill += n;
      if (lane == 0) sts_vol_i(sm.xfill, xfill);
      wd.start();
    } else {
      if (wd.expired(L)) return false;
      __nanosleep(256);
    }
  }
  return true;
}

template <int K, int WARPS, int D, int U, bool PRMT, bool LOCAL = false, bool CL = false>
__global__ void __launch_bounds__((WARPS + 2) * 32)
    nw_kernel(const SweepLaunch L, const PolSeq pol, const __grid_constant__ CUtensorMap tmap) {
  using S = NwSmem<K, WARPS, D, U>;
  extern __shared__ __align__(16) unsigned char nw_smem_raw[];
  const S sm(nw_smem_raw);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  (void)pol;
  if constexpr (CL) {
    // every CTA of a cluster runs the same rounds (cluster barriers must match)
    const int rounds = (L.nbands + gridDim.x - 1) / gridDim.x;
    bool failed = false;
    for (int round = 0; round < rounds; ++round) {
      const int band = blockIdx.x + round * gridDim.x;
      if (threadIdx.x < 64) reinterpret_cast<int*>(sm.wprog)[threadIdx.x] = 0;
      __syncthreads();
      cluster_sync_all();   // the neighbour's rings are initialised before any DSMEM store
      if (band < L.nbands && !failed) {
        if (warp == WARPS + 1) {
          nw_x_warp<K, WARPS, D, U>(L, sm, lane);
        } else if (warp == WARPS) {
          nw_io_warp<K, WARPS, D, U, LOCAL, true>(L, sm, band, lane);
        } else {
          NwWarp<K, WARPS, D, U, PRMT, LOCAL, true> w(L, &tmap, sm, band, warp, lane);
          w.run();
        }
      }
      __syncthreads();
      failed = failed || run_failed(L);
      cluster_sync_all();   // no CTA leaves (or re-initialises) while a neighbour may still store into it
    }
    return;
  } else {
  for (int band = blockIdx.x; band < L.nbands; band += gridDim.x) {
    if (threadIdx.x < 64) reinterpret_cast<int*>(sm.wprog)[threadIdx.x] = 0;   // wprog, rprog, xneed, xfill
    __syncthreads();
    if (warp == WARPS + 1) {
      nw_x_warp<K, WARPS, D, U>(L, sm, lane);
    } else if (warp == WARPS) {
      nw_io_warp<K, WARPS, D, U, LOCAL>(L, sm, band, lane);
    } else {
      NwWarp<K, WARPS, D, U, PRMT, LOCAL> w(L, &tmap, sm, band, warp, lane);
      w.run();
    }
    __syncthreads();
    if (run_failed(L)) return;
  }
  }
}

}  // namespace wfk
