// wf_nw.cuh -- the sequence-comparison (Needleman-Wunsch) band sweep, specialised for
// the B200 issue pipeline.  Same band / lane / skew / LL-handoff model as
// wf_sweep.cuh (read that header first); the differences, each measured (profiles/):
//
//  * Compute warps issue NO global memory operations in the row loop.  One I/O warp per
//    CTA (a) stages the row codes x_i into a shared-memory x ring ahead of use, (b) feeds
//    the band's west column (column-0 boundary or the previous band's LL ring) into
//    compute warp 0's shared LL ring, and (c) forwards the last compute warp's east
//    column from shared memory to the next band's / next slab's global LL ring.  The
//    compute warps' only fence -- fence.proxy.async before each TMA store, which lowers
//    to MEMBAR.ALL.CTA -- therefore waits for shared-memory stores only.
//  * Every compute warp has the same shape: input LL ring hand[w], output LL ring
//    hand[w+1] (hand[WARPS] belongs to the I/O warp).  Lane 0's west inputs for the next
//    U-row block are prefetched one block ahead; LL tags are checked once per block.
//  * The row loop runs in blocks of U steps with one body: ramp-up and drain blocks carry
//    a per-lane "row in range" predicate, steady blocks do not.  (A separate slow path
//    for the ~32 ramp steps per warp used to cost ~10 us per warp in the band chain.)
//  * Each block's U finished rows (32*K columns of the warp) leave shared memory in one
//    TMA 2-D tensor store (UTMASTG); the tensor bounds clip ramp rows <= 0, drain rows
//    > rows and the ragged last band.
//  * The cell, with W entering last (R9):
//        s  = score(x_i, y_j)          PRMT byte lookup (alphabet <= 8) or ISETP+SEL
//        t1 = max(N + g, NW + s)       IADD + VIADDMNMX
//        H  = max(W + g, t1)           VIADDMNMX
#pragma once
#include <cuda.h>

#include "wf_cells.cuh"
#include "wf_sweep.cuh"

namespace wfk {

constexpr int kXRing = 4096;   // rows of x codes staged ahead in shared memory (power of 2)
constexpr int kXMirror = 64;   // bytes of the ring's head mirrored after its end
#ifndef WF_IO_SLEEP_BUSY
#define WF_IO_SLEEP_BUSY 100
#endif
#ifndef WF_IO_SLEEP_IDLE
#define WF_IO_SLEEP_IDLE 200
#endif
constexpr unsigned kIoSleepBusy = WF_IO_SLEEP_BUSY;   // ns between I/O-warp polls after progress
constexpr unsigned kIoSleepIdle = WF_IO_SLEEP_IDLE;   // ns between polls that found nothing

template <int D, int U>
__host__ __device__ constexpr int nw_ring_rows() {
  // rows pending in a warp's staging ring: 31D (lane skew) + U (block) + TMA stores in flight
  return (31 * D + 3 * U) <= 64 ? 64 : (31 * D + 3 * U) <= 128 ? 128 : 256;
}

template <int K, int WARPS, int D, int U>
struct NwSmem {
  static constexpr int R = nw_ring_rows<D, U>();
  static constexpr int ROWB = 32 * K * 4;                                  // bytes per staged row
  static constexpr size_t stage_bytes = size_t(WARPS) * R * ROWB;
  static constexpr size_t hand_bytes = size_t(WARPS + 1) * kHandSlots * 8;
  static constexpr size_t ctl_bytes = 64 * 4;
  static constexpr size_t bytes = 1024 + stage_bytes + hand_bytes + kXRing + kXMirror + ctl_bytes;
  unsigned char* stage;     // 1024-byte aligned (TMA source rows)
  unsigned long long* hand; // [WARPS+1][kHandSlots] LL words
  unsigned char* xring;     // [kXRing] row codes, x of row r at (r-1) & (kXRing-1)
  int* prog;                // prog[w]: rows of hand[w] consumed by its reader (w = 0..WARPS)
  int* xneed;               // xneed[w]: lowest row warp w may still read from the x ring
  int* xfill;               // rows 1..*xfill of the x ring are valid
  __device__ __forceinline__ explicit NwSmem(unsigned char* raw) {
    const uint32_t a = static_cast<uint32_t>(__cvta_generic_to_shared(raw));
    unsigned char* base = raw + ((1024u - (a & 1023u)) & 1023u);
    stage = base;
    hand = reinterpret_cast<unsigned long long*>(base + stage_bytes);
    xring = base + stage_bytes + hand_bytes;
    prog = reinterpret_cast<int*>(xring + kXRing + kXMirror);
    xneed = prog + 16;
    xfill = prog + 32;
  }
  __device__ __forceinline__ unsigned long long* hand_slot(int w, int row) const {
    return hand + (size_t(w) * kHandSlots + (row & (kHandSlots - 1)));
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
__device__ __forceinline__ void sts_v2_u64(unsigned long long* p, unsigned long long a, unsigned long long b) {
  asm volatile("st.volatile.shared.v2.u64 [%0], {%1, %2};" ::"r"(static_cast<uint32_t>(__cvta_generic_to_shared(p))),
               "l"(a), "l"(b)
               : "memory");
}
__device__ __forceinline__ uint32_t lds_u8(const unsigned char* p) {
  uint32_t v;
  asm volatile("ld.volatile.shared.u8 %0, [%1];" : "=r"(v) : "r"(static_cast<uint32_t>(__cvta_generic_to_shared(p))));
  return v;
}

// =====================================================================================
// Compute warp: lane l owns K adjacent columns; at step t it is on row t - D*l + 1.
// =====================================================================================
template <int K, int WARPS, int D, int U, bool PRMT>
struct NwWarp {
  using S = NwSmem<K, WARPS, D, U>;
  static constexpr int R = S::R;
  static constexpr int ROWB = S::ROWB;
  // TMA groups that may still be reading the staging ring when a block starts writing it
  static constexpr int kMinDone = (R - U - 31 * D + 1 + U - 1) / U;   // ceil((R-U-31D+1)/U)
  static constexpr int kInFlight = kMinDone - 1;
  static_assert(kInFlight >= 0, "staging ring too small for the lane skew");
  static_assert(U % 2 == 0 && kHandSlots % U == 0 && R % U == 0, "block alignment");
#ifndef WF_NW_ABL
#define WF_NW_ABL 0
#endif
  // ablation switches for performance archaeology only (tools/ablate.sh); 0 in real builds
  static constexpr int kAbl = WF_NW_ABL;

  const SweepLaunch& L;
  const CUtensorMap* tmap;
  const S& sm;
  const int band, warp, lane;
  int rows;
  int32_t gap, mmatch, mmis;
  uint32_t qlo[K], qhi[K];   // PRMT: byte c = score(c, y_j) (int8) for c = 0..7
  uint32_t ycode[K];         // compare/select path
  int32_t Np[K];             // previous row at the lane's K columns
  int32_t prevW;             // previous row's west input (NW of the first column)
  int32_t q[D];              // east values of lane-1; q[D-1] is this step's west input
  int wcol;                  // warp's first column, slab-relative
  unsigned char* stage_lane; // staging ring + lane's segment
  uint32_t stage_w_s;        // shared address of this warp's staging ring
  int seen_prog_next;
  Watchdog wd;

  __device__ __forceinline__ NwWarp(const SweepLaunch& L_, const CUtensorMap* tmap_, const S& sm_, int band_,
                                    int warp_, int lane_)
      : L(L_), tmap(tmap_), sm(sm_), band(band_), warp(warp_), lane(lane_) {
    rows = L.rows;
    gap = L.gap;
    mmatch = L.match;
    mmis = L.mismatch;
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
      Np[m] = vc ? (jb + m + 1) * gap : 0;          // H[0][j] = j*g
    }
    prevW = jb < L.c1 ? jb * gap : 0;               // H[0][jb]
#pragma unroll
    for (int d = 0; d < D; ++d) q[d] = 0;
    unsigned char* stage_w = sm.stage + size_t(warp) * R * ROWB;
    stage_lane = stage_w + lane * (4 * K);
    stage_w_s = static_cast<uint32_t>(__cvta_generic_to_shared(stage_w));
    seen_prog_next = 0;
  }

  __device__ __forceinline__ void cells(int32_t Win, uint32_t xc, int32_t (&H)[K]) const {
    const uint32_t sel = xc * 0x1111u + 0x8880u;   // byte xc, sign-replicated (prmt default mode)
#pragma unroll
    for (int m = 0; m < K; ++m) {
      const int32_t NW = m == 0 ? prevW : Np[m - 1];
      const int32_t W = m == 0 ? Win : H[m - 1];
      int32_t s;
      if constexpr (PRMT) s = prmt_s8(qlo[m], qhi[m], sel);
      else s = (xc == ycode[m]) ? mmatch : mmis;
      const int32_t t1 = __viaddmax_s32(Np[m], gap, NW + s);
      H[m] = __viaddmax_s32(W, gap, t1);
    }
  }

  __device__ __forceinline__ void stage_store(int row, const int32_t (&H)[K]) const {
    unsigned char* dst = stage_lane + (row & (R - 1)) * ROWB;
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

  // plain copy of the finished row r from the staging ring to HBM (first block only)
  __device__ __forceinline__ void write_row(int r) const {
    const int jrel = wcol + lane * K;
    const int width = L.c1 - L.c0;
    const uint32_t* src = reinterpret_cast<const uint32_t*>(stage_lane + (r & (R - 1)) * ROWB);
    uint32_t* dst = static_cast<uint32_t*>(L.out[0]) + int64_t(r - 1) * L.pitch + jrel;
#pragma unroll
    for (int m = 0; m < K; ++m)
      if (jrel + m < width) dst[m] = src[m];
  }

  // Lane 0's west inputs for rows r0 .. r0+U-1: lane u (< U) loads the LL word of row r0+u
  // (one shared load for the whole block); lane 0 later takes its value by shuffle.
  __device__ __forceinline__ void load_west(int r0, int32_t& wv, uint32_t& wt) const {
    if (lane < U) {
      const unsigned long long v = lds_vol(sm.hand_slot(warp, r0 + lane));
      wv = static_cast<int32_t>(static_cast<uint32_t>(v));
      wt = static_cast<uint32_t>(v >> 32);
    }
  }
  __device__ __forceinline__ bool west_ok(int r0, uint32_t wt) const {
    const int r = r0 + lane;
    return __all_sync(0xffffffffu, lane >= U || r < 1 || r > rows || wt == static_cast<uint32_t>(r));
  }

  // room in hand[warp+1] for rows up to r_last (its reader publishes prog[warp+1])
  __device__ __forceinline__ bool room_next(int r_last) {
    const int need = r_last - kHandSlots;
    if (seen_prog_next >= need) return true;
    wd.start();
    for (;;) {
      seen_prog_next = lds_vol_i(sm.prog + warp + 1);
      if (seen_prog_next >= need) return true;
      if (wd.expired(L)) return false;
      __nanosleep(64);
    }
  }

  // x codes of rows [lo, hi] must be staged (I/O warp publishes *xfill)
  __device__ __forceinline__ bool x_ready(int hi, int& seen_xfill) {
    if (hi > rows) hi = rows;
    if (seen_xfill >= hi) return true;
    wd.start();
    for (;;) {
      seen_xfill = lds_vol_i(sm.xfill);
      if (seen_xfill >= hi) {
        __threadfence_block();   // order the x-ring reads after the observed fill count
        return true;
      }
      if (wd.expired(L)) return false;
      __nanosleep(32);
    }
  }

  template <bool EDGE>
  __device__ __forceinline__ void block(int t0, int32_t wv, const uint32_t (&xc)[U], int32_t (&east)[U]) {
#pragma unroll
    for (int u = 0; u < U; ++u) {
      const int row = t0 + u - D * lane + 1;
      const int32_t w0 = __shfl_sync(0xffffffffu, wv, u);       // lane 0's west input (row t0+u+1)
      const int32_t Win = (lane == 0) ? w0 : q[D - 1];
      int32_t H[K];
      cells(Win, xc[u], H);
      const bool active = !EDGE || (row >= 1 && row <= rows);
      if (active) {
        prevW = Win;
#pragma unroll
        for (int m = 0; m < K; ++m) Np[m] = H[m];
        stage_store(row, H);
      }
      east[u] = Np[K - 1];
      const int32_t r = __shfl_up_sync(0xffffffffu, Np[K - 1], 1);
#pragma unroll
      for (int d = D - 1; d > 0; --d) q[d] = q[d - 1];
      q[0] = r;
    }
  }

  // x codes of this lane's rows for the block starting at step t: rows t+u-D*lane+1, u < U.
  // The x ring has a mirrored tail of kXMirror bytes, so the U loads use immediate offsets.
  __device__ __forceinline__ void load_x(int t, uint32_t (&xo)[U]) const {
    const unsigned char* p = sm.xring + ((t - D * lane) & (kXRing - 1));
#pragma unroll
    for (int u = 0; u < U; ++u) xo[u] = lds_u8(p + u);
  }

  __device__ __forceinline__ bool run() {
    const int T = rows + 31 * D;                  // steps
    // blocks start at t0 == 31D-1 (mod U): lane 31's rows of a block, r31_0 = t0-31D+1, are
    // a multiple of U (aligned TMA boxes and 16-byte LL pairs)
    int t0 = (31 * D - 1) % U;
    if (t0 > 0) t0 -= U;
    const int steady_lo = 31 * D;                 // t >= 31D: lane 31's row >= 1
    const int steady_hi = rows - U;               // t0 + U - 1 <= rows - 1: lane 0's row <= rows
    const bool tracing = L.trace != nullptr && warp == 0 && lane == 0;
    const int trace_every = (rows + kTraceRows - 1) / kTraceRows;
    int trace_next = trace_every;
    if (tracing) {
      L.trace[size_t(band) * kTraceSlots] = globaltimer();
      L.trace[size_t(band) * kTraceSlots + 42] = clock64();
    }
    int seen_xfill = 0;
    // prefetch block 0's west inputs and row codes
    int32_t wvn = 0;
    uint32_t wtn = 0;
    uint32_t xn[U];
    if (!x_ready(t0 + U + U, seen_xfill)) return false;
    load_west(t0 + 1, wvn, wtn);
    load_x(t0, xn);
#ifdef WF_PHASE_PROF
    long long ph_acc[8] = {0, 0, 0, 0, 0, 0, 0, 0};
    long long ph_last = clock64();
#define WF_PH(i)                                   \
  do {                                             \
    const long long now_ = clock64();              \
    ph_acc[(i)] += now_ - ph_last;                 \
    ph_last = now_;                                \
  } while (0)
#else
#define WF_PH(i) \
  do {           \
  } while (0)
#endif
    for (; t0 < T; t0 += U) {
      if (tracing && t0 >= trace_next) {
        L.trace[size_t(band) * kTraceSlots + (t0 / trace_every < kTraceRows ? t0 / trace_every : kTraceRows - 1)] =
            globaltimer();
        trace_next += trace_every;
      }
      WF_PH(0);
      // ---- this block's inputs (validated), next block's prefetched
      int32_t wv = wvn;
      uint32_t xc[U];
#pragma unroll
      for (int u = 0; u < U; ++u) xc[u] = xn[u];
      if (!(kAbl & 2) && !west_ok(t0 + 1, wtn)) {
        wd.start();
        for (;;) {
          uint32_t wt = 0;
          load_west(t0 + 1, wv, wt);
          if (west_ok(t0 + 1, wt)) break;
          if (wd.expired(L)) return false;
          __nanosleep(20);
        }
      }
      if (lane == 0) {
        sts_vol_i(sm.prog + warp, t0 + U);        // rows <= t0+U of hand[warp] consumed
        sts_vol_i(sm.xneed + warp, t0 - 31 * D + 1);
      }
      WF_PH(1);
      if (!(kAbl & 32) && !x_ready(t0 + 3 * U, seen_xfill)) return false;
      if (!(kAbl & 4)) load_x(t0 + U, xn);
      WF_PH(2);
      // ---- ring slots about to be overwritten must have been read by older TMA stores
      if (!(kAbl & 8)) {
        if (lane == 0) bulk_wait_read<kInFlight>();
        __syncwarp();
      }
      const int r31_0 = t0 - 31 * D + 1;           // multiple of U
      if (!(kAbl & 64) && !room_next(r31_0 + U - 1)) return false;
      WF_PH(3);
      int32_t east[U];
      if (t0 >= steady_lo && t0 <= steady_hi) block<false>(t0, wv, xc, east);
      else block<true>(t0, wv, xc, east);
      WF_PH(4);
      // ---- lane 31 publishes its east column for rows r31_0 .. r31_0+U-1
      if (!(kAbl & 16) && lane == 31 && r31_0 + U - 1 >= 1 && r31_0 <= rows) {
        unsigned long long* s = sm.hand_slot(warp + 1, r31_0);
#pragma unroll
        for (int u = 0; u < U; u += 2)
          sts_v2_u64(s + u, ll_pack(static_cast<uint32_t>(east[u]), static_cast<uint32_t>(r31_0 + u)),
                     ll_pack(static_cast<uint32_t>(east[u + 1]), static_cast<uint32_t>(r31_0 + u + 1)));
      }
      WF_PH(5);
      // ---- the block's finished rows leave shared memory by one TMA store (clipped at the
      //      drain end and the ragged band; a negative start row is not a legal TMA store
      //      coordinate, so the first block -- rows 0..U-1 -- uses plain stores)
      if ((kAbl & 1) == 0 && r31_0 >= 1 && r31_0 <= rows) {
        fence_proxy_async_smem();
        __syncwarp();
        if (lane == 0) {
          tma_store_2d(tmap, stage_w_s + (r31_0 & (R - 1)) * ROWB, wcol, r31_0 - 1);
          bulk_commit();
        }
      } else if (r31_0 + U - 1 >= 1 && r31_0 <= rows) {
        __syncwarp();
        for (int r = max(r31_0, 1); r <= min(r31_0 + U - 1, rows); ++r) write_row(r);
      }
      WF_PH(6);
      // ---- next block's west inputs: read as late as possible so the producer (previous
      //      warp / I/O warp) has had this whole block to publish them
      if (!(kAbl & 2)) load_west(t0 + U + 1, wvn, wtn);
      WF_PH(7);
    }
#ifdef WF_PHASE_PROF
    if (tracing)
      for (int i = 0; i < 8; ++i) L.trace[size_t(band) * kTraceSlots + 44 + i] = static_cast<unsigned long long>(ph_acc[i]);
#endif
    if (lane == 0) bulk_wait_all();
    if (lane == 0) sts_vol_i(sm.xneed + warp, rows + 1);
    if (tracing) {
      L.trace[size_t(band) * kTraceSlots + kTraceRows] = globaltimer();
      L.trace[size_t(band) * kTraceSlots + 43] = clock64();
    }
    return true;
  }
};

// =====================================================================================
// I/O warp: x staging, west feed of warp 0, east forwarding of warp WARPS-1.
// =====================================================================================
template <int K, int WARPS, int D, int U>
__device__ __forceinline__ bool nw_io_warp(const SweepLaunch& L, const NwSmem<K, WARPS, D, U>& sm, int band,
                                           int lane) {
  const int rows = L.rows;
  const uint8_t* x = static_cast<const uint8_t*>(L.row_in);
  const bool boundary = L.first_slab && band == 0;
  const unsigned long long* src = L.edge + size_t(band) * edge_stride(rows);                 // inbound ring
  unsigned long long* dst = (band + 1 < L.nbands) ? L.edge + size_t(band + 1) * edge_stride(rows) : L.next_edge;
  const bool wait_ack = band + 1 >= L.nbands && L.next_edge && L.ack_self;
  int xfill = 0;                // rows 1..xfill staged
  int feed = 1;                 // next row to feed into hand[0]
  int fwd = 1;                  // next row to forward from hand[WARPS]
  int seen_prog0 = 0;
  bool acked = !wait_ack;
  Watchdog wd;
  wd.start();
  while (xfill < rows || feed <= rows || fwd <= rows) {
    bool progress = false;
    // (a) x ring: keep up to kXRing rows ahead of the slowest compute warp
    if (xfill < rows) {
      int lo = rows + 1;
#pragma unroll
      for (int w = 0; w < WARPS; ++w) lo = min(lo, lds_vol_i(sm.xneed + w));
      const int cap = min(rows, lo - 1 + kXRing);
      if (cap > xfill) {
        const int n = min(cap - xfill, 512);
        for (int i = lane; i < n; i += 32) {
          const int r = xfill + 1 + i;
          const int slot = (r - 1) & (kXRing - 1);
          const unsigned char xv = __ldg(x + (r - 1));
          sm.xring[slot] = xv;
          if (slot < kXMirror) sm.xring[kXRing + slot] = xv;   // mirrored head
        }
        __syncwarp();
        __threadfence_block();
        xfill += n;
        if (lane == 0) sts_vol_i(sm.xfill, xfill);
        progress = true;
      }
    }
    // (b) west feed of compute warp 0 (boundary column or the previous band's LL ring)
    if (feed <= rows) {
      const int need = feed + 63 - kHandSlots;    // slot reuse: hand[0] rows consumed
      if (seen_prog0 < need) seen_prog0 = lds_vol_i(sm.prog + 0);
      if (seen_prog0 >= need) {
        uint32_t v[2];
        bool ok[2];
#pragma unroll
        for (int h = 0; h < 2; ++h) {
          const int r = feed + h * 32 + lane;
          ok[h] = true;
          v[h] = 0;
          if (r <= rows) {
            if (boundary) {
              v[h] = static_cast<uint32_t>(r * L.gap);          // H[r][0] = r*g
            } else {
              const unsigned long long wv = ld_relaxed_sys(src + r);
              v[h] = static_cast<uint32_t>(wv);
              ok[h] = static_cast<uint32_t>(wv >> 32) == L.epoch;
            }
          }
        }
        const unsigned m0 = __ballot_sync(0xffffffffu, ok[0]);
        const unsigned m1 = __ballot_sync(0xffffffffu, ok[1]);
        int n = (m0 == 0xffffffffu) ? 32 + (__ffs(~m1) ? __ffs(~m1) - 1 : 32) : __ffs(~m0) - 1;
        if (feed + n > rows + 1) n = rows + 1 - feed;
#pragma unroll
        for (int h = 0; h < 2; ++h) {
          const int r = feed + h * 32 + lane;
          if (r < feed + n) sts_vol(sm.hand_slot(0, r), ll_pack(v[h], static_cast<uint32_t>(r)));
        }
        if (n > 0) progress = true;
        feed += n;
        if (feed > rows && !L.first_slab && band == 0 && L.ack_prev && lane == 0)
          st_relaxed_sys_u32(L.ack_prev, L.epoch);   // predecessor slab may reuse this ring
      }
    }
    // (c) forward the band's east column from hand[WARPS] to the next band / slab
    if (fwd <= rows) {
      if (!acked) {   // the next slab must have drained its ring in the previous run
        const unsigned a = ld_relaxed_sys_u32(L.ack_self);
        acked = static_cast<int>(a - (L.epoch - 1u)) >= 0;
      }
      if (acked) {
        const int r = fwd + lane;
        bool ok = true;
        uint32_t v = 0;
        if (r <= rows) {
          const unsigned long long wv = lds_vol(sm.hand_slot(WARPS, r));
          v = static_cast<uint32_t>(wv);
          ok = static_cast<uint32_t>(wv >> 32) == static_cast<uint32_t>(r);
        }
        const unsigned m = __ballot_sync(0xffffffffu, ok);
        int n = (m == 0xffffffffu) ? 32 : __ffs(~m) - 1;
        if (fwd + n > rows + 1) n = rows + 1 - fwd;
        if (r < fwd + n && dst) st_relaxed_sys(dst + r, ll_pack(v, L.epoch));
        if (n > 0) {
          fwd += n;
          if (lane == 0) sts_vol_i(sm.prog + WARPS, fwd - 1);
          progress = true;
        }
      }
    }
    // The I/O warp only needs to stay a few blocks ahead; polling at full rate would steal
    // the SM's MIO pipe (shared-memory / shuffle issue) from the compute warps.
    if (progress) {
      wd.start();
      __nanosleep(kIoSleepBusy);
    } else {
      if (wd.expired(L)) return false;
      __nanosleep(kIoSleepIdle);
    }
  }
  return true;
}

template <int K, int WARPS, int D, int U, bool PRMT>
__global__ void __launch_bounds__((WARPS + 1) * 32)
    nw_kernel(const SweepLaunch L, const PolSeq pol, const __grid_constant__ CUtensorMap tmap) {
  using S = NwSmem<K, WARPS, D, U>;
  extern __shared__ __align__(16) unsigned char nw_smem_raw[];
  const S sm(nw_smem_raw);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  (void)pol;
  for (int band = blockIdx.x; band < L.nbands; band += gridDim.x) {
    for (int i = threadIdx.x; i < (WARPS + 1) * kHandSlots; i += blockDim.x) sm.hand[i] = 0ull;
    if (threadIdx.x < 64) sm.prog[threadIdx.x] = 0;    // prog, xneed, xfill
    __syncthreads();
    if (warp == WARPS) {
      nw_io_warp<K, WARPS, D, U>(L, sm, band, lane);
    } else {
      NwWarp<K, WARPS, D, U, PRMT> w(L, &tmap, sm, band, warp, lane);
      w.run();
    }
    __syncthreads();
    if (run_failed(L)) return;
  }
}

}  // namespace wfk
