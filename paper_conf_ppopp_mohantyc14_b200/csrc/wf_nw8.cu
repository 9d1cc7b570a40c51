// wf_nw8.cu -- sequence comparison (Needleman-Wunsch; Smith-Waterman,
// P:732) band sweep, generation 8: one long lane pipeline.
//
// Why a new generation.  The v4 kernel (wf_nw.cuh) ran 2 compute warps per SM with 32-row
// block hand-offs; its time was (rows + 127 band hops x ~222 rows) x 87 cycles -- the hops,
// not the cells (profiles/r01_microbench.txt).  The critical path of the sweep
// is the chain of hand-offs, so v8 makes every hand-off cost about one row:
//
//  * Every lane of every warp of every CTA is one stage of a single skewed pipeline over the
//    slab's columns: lane l of a warp owns K adjacent columns and at local step s is on row
//    s - l (the paper's "within a diagonal, computation of each data point is independent",
//    P:193-200, without per-diagonal launches).  T ~= (rows + lanes + hand-off excess) x step.
//  * WARPS compute warps per CTA (4 = one per SM sub-partition), K = 2, plus one helper warp
//    that owns all global-memory hand-off traffic; the row codes are copied to shared memory
//    once per CTA.
//  * Lane -> lane: SHFL.IDX rotation.  Lane 31's slot carries lane 0's NEXT west input, so the
//    only instructions on the lane-to-lane chain are SHFL and ONE VIADDMNMX:
//    E = max(W + K g, P_{K-1}) = H_{K-1} for lanes 0..30, max(W - 2^29, in) = in for lane 31.
//  * Warp -> warp inside a CTA: LOCKSTEP.  The warps of a CTA advance in blocks of U steps
//    separated by one named CTA barrier, warp w running LAG = 32 + U rows behind warp w-1.
//    Lane 31 of warp w-1 stores its east value of row r into a shared ring (plain int32, one
//    STS per step); by the lag, every word warp w needs in a block was stored before the
//    barrier that opens the block, so the reader loads U rows with U/4 broadcast 16-byte loads
//    and needs no flag, tag, sentinel or flow control (the barrier orders shared memory).
//    Every compute warp -- the first and the last included -- runs this one shared-ring role.
//  * Band -> band (CTA -> CTA) and slab -> slab (GPU -> GPU over NVLink): the helper warp, on
//    the same block clock (it joins the barrier).  Outbound, one block after the last compute
//    warp stored a block of east words into its shared ring, the helper forwards them with
//    16-byte stores into the next band's / next slab's global ring (slot r = row r; a peer /
//    IPC address at the slab edge).  Inbound, it loads the band's global words one block ahead
//    of warp 0, checks that none is the EMPTY sentinel (a stale quad spins on the global words;
//    the CTA then waits at the barrier), writes them into warp 0's shared ring and resets the
//    global slots to EMPTY for the next run (between slabs the reset is fenced before the
//    per-run ack the producer slab waits on).  (An asynchronous helper outside the barrier
//    measured slower: its polling competes with warp 0 for issue slots.)
//  * Outputs: per-warp staging ring (128 rows x 32K int32, row-major) -> one TMA 2-D tensor
//    store (UTMASTG) per 32 rows; every output byte is written to HBM exactly once.
//  * Cell (W enters last, R9), prefix form:
//        s_m = (x_i == y_j) ? match : mismatch                      ISETP + SEL
//        t_m = max(N_m + g, NW_m + s_m)            (SW: and 0)      IADD + VIADDMNMX(.RELU)
//        P_m = max(t_m, P_{m-1} + g)                                VIADDMNMX
//        H_m = max(P_m, W + (m+1) g)                                VIADDMNMX
//    = max(t_m, H_{m-1} + g) unrolled along the lane's row (same integer).
#include <cstdio>
#include <cstring>

#include <cuda.h>
#include <cudaTypedefs.h>

#include "wf_nw.cuh"
#include "wf_sweep.cuh"
#include "wf_variant.h"

namespace wfk {

cudaError_t encode_plane_map(CUtensorMap* m, const SweepLaunch& L, int box_cols, int box_rows);
cudaError_t encode_map_2d(CUtensorMap* m, void* base, int cols, int rows, int64_t pitch_elems, int box_cols, int box_rows);

namespace nw8 {

#ifndef WF_NW8_U
#define WF_NW8_U 16    // steps per lockstep block (A/B: 8 and 4 slower, profiles/r02_nw8_ab.txt)
#endif
#ifndef WF_NW8_HELPER_TMA
// who issues the compute warps' TMA output stores: 0 = each compute warp's lane 0, 1 = the
// helper warp, 2 = a separate storer warp (on another SM sub-partition than the helper)
#define WF_NW8_HELPER_TMA 2
#endif
constexpr int kExtraWarps = WF_NW8_HELPER_TMA == 2 ? 2 : 1;   // warps besides the compute warps
#ifndef WF_NW8_DPRE_ROWS
#define WF_NW8_DPRE_ROWS 32  // rows ahead the helper loads the inbound words (profiles/r02_nw8_ab.txt)
#endif
#ifndef WF_NW8_DIRECT_EAST
#define WF_NW8_DIRECT_EAST 1   // the last compute warp stores its east words straight to the next band's ring
#endif

constexpr int RR = 128;        // slots per shared ring (power of 2, > 2U for every compiled U <= 32)
constexpr int SR = 128;        // staging rows per warp (power of 2, = 4 TMA boxes)
constexpr int XPAD = 64;       // bytes of padding around the shared x copy
constexpr int XMAX = 65536;    // rows the shared x copy holds (ABI maximum 65535)
constexpr unsigned FULL = 0xffffffffu;
constexpr int32_t EMPTY = static_cast<int32_t>(0x80808080u);   // memset(0x80) pattern; |H| < 2^24

// global ring of band b: int32 slots, row r at base[b * stride + kGOff + r]; 32+ slots of
// slack on each side; the stride is a multiple of 4 and kGOff = 2 mod 4, so rows r0 .. r0+3
// with r0 = 2 mod 4 are one aligned 16-byte quad.  Fits in the host's per-band allocation of
// (edge_stride + 64) u64 words.
constexpr int kGOff = 34;
__host__ __device__ inline size_t gring_stride(int rows) { return ((size_t(rows) + 5) & ~size_t(3)) + 64; }

// shared ring slot byte offset of row r: rows r0 .. r0+3 with r0 = 2 mod 4 are one aligned quad
__device__ __forceinline__ uint32_t slot(int r) { return uint32_t((r + 2) & (RR - 1)) * 4; }

template <int K, int WARPS>
struct Smem {
  static constexpr int ROWB = 32 * K * 4;   // bytes per staged row of one warp
  static constexpr size_t stage_bytes = size_t(WARPS) * SR * ROWB;
  static constexpr size_t ring_bytes = size_t(WARPS + 1) * RR * 4;
  static constexpr size_t x_bytes = XMAX + 2 * XPAD;
  static constexpr size_t ctl_bytes = 128;
  static constexpr size_t bytes = 1024 + stage_bytes + ring_bytes + x_bytes + ctl_bytes;
  unsigned char* stage;   // [WARPS][SR][32K] int32 (TMA source), 1024-byte aligned
  int32_t* ring;          // [WARPS+1][RR]: ring w = west words of compute warp w (ring 0: from the
                          // helper), ring WARPS = east words of the last compute warp (to the helper)
  unsigned char* x;       // x[r - 1] = code of row r, r = 1..rows (XPAD bytes of slack each side)
  int* ctl;               // ctl[31] = EMPTY (read back as a register value)
  __device__ __forceinline__ explicit Smem(unsigned char* raw) {
    const uint32_t a = static_cast<uint32_t>(__cvta_generic_to_shared(raw));
    unsigned char* base = raw + ((1024u - (a & 1023u)) & 1023u);
    stage = base;
    ring = reinterpret_cast<int32_t*>(base + stage_bytes);
    x = base + stage_bytes + ring_bytes + XPAD;
    ctl = reinterpret_cast<int*>(base + stage_bytes + ring_bytes + x_bytes);
  }
};

__device__ __forceinline__ uint32_t saddr(const void* p) { return static_cast<uint32_t>(__cvta_generic_to_shared(p)); }

__device__ __forceinline__ int4 lds128(uint32_t a) {
  int4 v;
  asm volatile("ld.volatile.shared.v4.s32 {%0, %1, %2, %3}, [%4];" : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "r"(a));
  return v;
}
__device__ __forceinline__ void sts128(uint32_t a, const int4& v) {
  asm volatile("st.shared.v4.s32 [%0], {%1, %2, %3, %4};" ::"r"(a), "r"(v.x), "r"(v.y), "r"(v.z), "r"(v.w));
}
__device__ __forceinline__ int4 ldg128_sys(const int32_t* p) {
  int4 v;
  asm volatile("ld.volatile.global.v4.s32 {%0, %1, %2, %3}, [%4];"
               : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w)
               : "l"(p)
               : "memory");
  return v;
}
__device__ __forceinline__ int32_t ldg32_sys(const int32_t* p) {
  int32_t v;
  asm volatile("ld.relaxed.sys.global.s32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void stg32_sys(int32_t* a, int32_t v) {
  asm volatile("st.volatile.global.s32 [%0], %1;" ::"l"(a), "r"(v) : "memory");
}
// 16-byte global stores of the hand-off: each of the four 4-byte words is single-copy atomic,
// the consumer checks every word
__device__ __forceinline__ void stg128_sys(int32_t* a, const int4& v) {
  asm volatile("st.volatile.global.v4.s32 [%0], {%1, %2, %3, %4};" ::"l"(a), "r"(v.x), "r"(v.y), "r"(v.z), "r"(v.w)
               : "memory");
}
__device__ __forceinline__ int32_t lds32(uint32_t a) {
  int32_t v;
  asm volatile("ld.volatile.shared.s32 %0, [%1];" : "=r"(v) : "r"(a) : "memory");
  return v;
}
// predicated store: a divergent `if (lane == 31)` would wrap the following shuffles in a
// reconvergence sequence
__device__ __forceinline__ void stg128_if(bool p, int32_t* a, const int4& v) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %5, 0; @q st.volatile.global.v4.s32 [%0], {%1, %2, %3, %4}; }" ::"l"(a),
               "r"(v.x), "r"(v.y), "r"(v.z), "r"(v.w), "r"(static_cast<int>(p)));
}
__device__ __forceinline__ void stg32_if(bool p, int32_t* a, int32_t v) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q st.volatile.global.s32 [%0], %1; }" ::"l"(a), "r"(v),
               "r"(static_cast<int>(p)));
}
__device__ __forceinline__ void sts32_if(bool p, uint32_t a, int32_t v) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q st.shared.s32 [%0], %1; }" ::"r"(a), "r"(v),
               "r"(static_cast<int>(p)));
}
// The block barrier.  The warps reach it from different code (each warp's role is its own
// instantiation), as in warp-specialized producer / consumer kernels: each warp arrives
// convergently, the CTA's warps at different barrier instructions.  bar.sync (the .aligned
// form) measured 7 % faster on C4 than barrier.sync (1.962 vs 2.101 ms, profiles/r02_nw8_ab.txt);
// compute-sanitizer synccheck reports the .aligned form as "divergent threads in block", so the
// sanitizer runs build the non-.aligned form (-DWF_NW8_UNALIGNED_BAR, tools/gpu_race.sh), which is
// synccheck-clean and passes the same parity (profiles/r02_sanitizer.txt).
template <int THREADS>
__device__ __forceinline__ void cta_bar() {
#ifdef WF_NW8_UNALIGNED_BAR
  asm volatile("barrier.sync 1, %0;" ::"n"(THREADS) : "memory");
#else
  asm volatile("bar.sync 1, %0;" ::"n"(THREADS) : "memory");
#endif
}
__device__ __forceinline__ bool quad_stale(const int4& v, int r, int rows) {
  return (v.x == EMPTY && r <= rows) | (v.y == EMPTY && r + 1 <= rows) | (v.z == EMPTY && r + 2 <= rows) |
         (v.w == EMPTY && r + 3 <= rows);
}

// ---------------------------------------------------------------------------------------------
// One compute warp: warp index WI of the CTA.  BOUND: lane 0's west inputs are the column-0
// boundary (first band of the first slab); otherwise they come from shared ring WI (written by
// warp WI-1, or for WI = 0 by the helper warp).  Lane 31's east words go to shared ring WI + 1
// (for the last warp: the helper's outbound ring).  U: steps per lockstep block.
// ---------------------------------------------------------------------------------------------
template <int K, int WARPS, int WI, bool BOUND, bool LOCAL, int U>
struct Warp {
  using S = Smem<K, WARPS>;
  static constexpr int ROWB = S::ROWB;
  static constexpr int LAG = 32 + U;   // rows between consecutive warps (lockstep)
  static constexpr int NT = (WARPS + kExtraWarps) * 32;   // threads at the CTA barrier (compute + helper warps)
  static_assert(U % 4 == 0 && 32 % U == 0, "block of U steps: multiple of 4, divides 32");
  static_assert(RR > 2 * U, "ring size");
  static_assert(SR * ROWB <= 65536, "staging slot arithmetic");

  const SweepLaunch& L;
  const CUtensorMap* tmap;   // this band's output map: the slab's plane, or (NEXT-4 overlap bands) the scratch plane
  const int band, lane;
  const bool is31;
  int ocol;                  // this warp's first column in tmap's plane
  int rows;
  int32_t gap, mmatch, mmis;
  int32_t gk[K];          // (m+1) g
  int32_t gLx;            // lane 31: -2^29 (E = its next west input); others K g
  uint32_t ycode[K];      // the lane's column codes
  int32_t N[K];           // H of the lane's previous row
  int32_t NWc;            // previous row's west input (NW of the first column)
  int32_t src;            // value this lane hands on at the next shuffle
  int srcl;               // (lane + 31) & 31
  int wcol;               // warp's first column, slab-relative
  uint32_t stage_s;       // shared address of this warp's staging ring
  uint32_t lane_off;      // lane * 4K (byte offset of the lane's columns in a staged row)
  uint32_t ring_in;       // shared address of ring WI
  uint32_t ring_out;      // shared address of ring WI + 1
  int32_t* gout;          // last warp (WF_NW8_DIRECT_EAST): the next band's / slab's global ring, row r at gout[r]
  bool east_out;          // ... and there is one (not the last band of the last slab); lane 31 only
  int32_t* gx;            // NEXT-4 halo export band: the next slab's ring as a second destination
  bool east_x;
  int32_t east_last;      // last warp: lane 31's east word of the current step
  uint32_t x_s;           // shared address of the x copy (x of row r at x_s + r - 1)
  int32_t best = 0, best_row = 0;   // LOCAL: best cell value of the lane and the first row reaching it
  int32_t vrow;           // NW: r c of the lane's first virtual row r = -lane (0 for SW)

  __device__ __forceinline__ Warp(const SweepLaunch& L_, const CUtensorMap* tm, const CUtensorMap* tm_halo, const S& sm,
                                  int band_, int lane_)
      : L(L_), tmap(band_ < L_.halo_bands ? tm_halo : tm), band(band_), lane(lane_), is31(lane_ == 31) {
    rows = L.rows;
    gap = L.gap;
    mmatch = L.match;
    mmis = L.mismatch;
#pragma unroll
    for (int m = 0; m < K; ++m) gk[m] = (m + 1) * gap;
    gLx = is31 ? -(1 << 29) : K * gap;
    const uint8_t* y = static_cast<const uint8_t*>(L.col_in);
    wcol = band * L.band_w + WI * 32 * K;      // relative to the first computed column cc0
    ocol = band < L.halo_bands ? wcol : wcol - L.halo_bands * L.band_w;
    const int jb = L.cc0 + wcol + lane * K;   // global 0-based first column of the lane
    // NW: lane l starts at step 1 on row 1 - l.  Instead of predicating every state update of the
    // ramp-up steps (rows <= 0), the row-0 boundary is extended to virtual rows r <= 0 by
    // V(r, j) = j g + r c with c = max(1, g, max(match, mismatch) - g): V is a fixed point of the
    // recurrence (N + g <= V since g <= c; NW + s <= V since s - g <= c; W + g = V), so a lane
    // that starts from row -l's V values and receives V as its west input reproduces V on its
    // virtual rows and reaches row 0 = the true boundary, for any scores (
    // checked over the ABI scoring range by tests/test_nw_virtual_rows.py).
    // SW keeps the predicated ramp (its floor 0 has no such extension).
    const int32_t vc_ = max(1, max(gap, max(mmatch, mmis) - gap));
    vrow = LOCAL ? 0 : -lane * vc_;                                          // V(-lane, j) - j g
#pragma unroll
    for (int m = 0; m < K; ++m) {
      const bool vc = jb + m < L.c1;
      ycode[m] = vc ? static_cast<uint32_t>(__ldg(y + jb + m)) : 0x100u;   // never equal to a code
      N[m] = LOCAL ? 0 : (jb + m + 1) * gap + vrow;                         // H[0][j] = j g (NW; V(-lane, j)), 0 (SW)
    }
    NWc = (!LOCAL) ? jb * gap + vrow : 0;                                   // H[0][jb] (NW: V(-lane, jb))
    // what this lane hands its east neighbour at step 1: its east value of row -lane (NW: V)
    src = LOCAL ? 0 : (jb + K) * gap + vrow;
    srcl = (lane + 31) & 31;
    stage_s = saddr(sm.stage) + uint32_t(WI) * SR * ROWB;
    lane_off = uint32_t(lane) * 4 * K;
    ring_in = saddr(sm.ring) + uint32_t(WI) * RR * 4;
    ring_out = saddr(sm.ring) + uint32_t(WI + 1) * RR * 4;
    gout = nullptr;
    east_out = false;
    gx = nullptr;
    east_x = false;
    if (WF_NW8_DIRECT_EAST && WI == WARPS - 1) {
      int32_t* gbase = reinterpret_cast<int32_t*>(L.edge);
      gout = (band + 1 < L.nbands) ? gbase + size_t(band + 1) * gring_stride(rows) + kGOff
                                   : (L.next_edge && band == L.export_band ? reinterpret_cast<int32_t*>(L.next_edge) + kGOff
                                                                           : nullptr);
      // NEXT-4 halo: the export band also feeds the next slab (whose overlap starts after it)
      gx = (band + 1 < L.nbands && band == L.export_band && L.next_edge)
               ? reinterpret_cast<int32_t*>(L.next_edge) + kGOff : nullptr;
      east_out = gout != nullptr;
      east_out = east_out && is31;
      east_x = gx != nullptr && is31;
    }
    x_s = saddr(sm.x);
  }

  static __device__ __forceinline__ int32_t t1f(int32_t n, int32_t g, int32_t d) {
    if constexpr (LOCAL) return __viaddmax_s32_relu(n, g, d);   // max(n + g, d, 0)
    else return __viaddmax_s32(n, g, d);
  }

  // ---- one step (local step s) ------------------------------------------------------------
  template <bool EDGE>
  __device__ __forceinline__ void step(int s, uint32_t xc, int32_t in_next, uint32_t soff, uint32_t rout) {
    const int32_t W = __shfl_sync(FULL, src, srcl);   // lane 0: in[s]; lane l: lane l-1's east at row s-l
    int32_t P[K], H[K];
#pragma unroll
    for (int m = 0; m < K; ++m) {
      const int32_t sc = (xc == ycode[m]) ? mmatch : mmis;
      const int32_t nw = m == 0 ? NWc : N[m - 1];
      const int32_t tm = t1f(N[m], gap, nw + sc);
      P[m] = m == 0 ? tm : __viaddmax_s32(P[m - 1], gap, tm);
    }
    const int32_t Px = is31 ? in_next : P[K - 1];
    src = __viaddmax_s32(W, gLx, Px);   // lanes 0..30: H[K-1]; lane 31: lane 0's next west input
#pragma unroll
    for (int m = 0; m < K; ++m) H[m] = __viaddmax_s32(W, gk[m], P[m]);
    const int row = s - lane;
    // staging: slot (row - 1) mod SR.  soff = (row - 1) * ROWB (mod 2^32); rows <= 0 land in
    // slots rewritten before their box is stored; rows > rows are clipped by the tensor bounds
    const uint32_t a = stage_s + ((soff & uint32_t(SR * ROWB - 1)) | lane_off);
    if constexpr (K == 1) {
      asm volatile("st.shared.b32 [%0], %1;" ::"r"(a), "r"(H[0]));
    } else if constexpr (K == 2) {
      asm volatile("st.shared.v2.b32 [%0], {%1, %2};" ::"r"(a), "r"(H[0]), "r"(H[1]));
    } else {
#pragma unroll
      for (int m = 0; m < K; m += 4)
        asm volatile("st.shared.v4.b32 [%0], {%1, %2, %3, %4};" ::"r"(a + 4 * m), "r"(H[m]), "r"(H[m + 1]),
                     "r"(H[m + 2]), "r"(H[m + 3]));
    }
    bool active = true;
    if constexpr (EDGE) active = row >= 1 && row <= rows;
    if (WF_NW8_DIRECT_EAST && WI == WARPS - 1) {
      east_last = H[K - 1];   // block() stores 4 rows at a time into the next band's ring
    } else {
      sts32_if(is31 && active, rout, H[K - 1]);   // east hand-off: lane 31's row s - 31
    }
    if constexpr (LOCAL) {   // best cell: strict > keeps the first row reaching the value
      int32_t rm = H[0];
#pragma unroll
      for (int m = 1; m < K; ++m) rm = max(rm, H[m]);
      const bool up = rm > best && active;
      best = up ? rm : best;
      best_row = up ? row : best_row;
    }
    if constexpr (EDGE) {
      NWc = active ? W : NWc;
#pragma unroll
      for (int m = 0; m < K; ++m) N[m] = active ? H[m] : N[m];
    } else {
      NWc = W;
#pragma unroll
      for (int m = 0; m < K; ++m) N[m] = H[m];
    }
  }

  // x codes of the lane's rows at local steps s0+1 .. s0+U (x of row r at x_s + r - 1)
  __device__ __forceinline__ void load_x(int s0, uint32_t (&xc)[U]) const {
    const uint32_t xb = x_s + uint32_t(s0 - lane);
#pragma unroll
    for (int u = 0; u < U; ++u) asm volatile("ld.shared.u8 %0, [%1];" : "=r"(xc[u]) : "r"(xb + uint32_t(u)));
  }

  // ---- one block: local steps s0+1 .. s0+U (after the barrier that opens it) ----------------
  // xc holds the x codes of this block on entry and those of the next block on exit (each is
  // reloaded right after its step used it, so the load latency hides behind the block)
  template <bool EDGE>
  __device__ __forceinline__ void block(int s0, uint32_t (&xc)[U]) {
    int32_t in[U];
    const int r0 = s0 + 2;   // rows of lane 31's next west inputs: r0 .. r0+U-1
    if constexpr (BOUND) {
#pragma unroll
      for (int u = 0; u < U; ++u) in[u] = LOCAL ? 0 : (r0 + u) * gap;
    } else {
      // stored by warp WI-1 (or the helper) before the barrier that opened this block
#pragma unroll
      for (int q = 0; q < U / 4; ++q) {
        const int4 v = lds128(ring_in + slot(r0 + 4 * q));
        in[4 * q] = v.x;
        in[4 * q + 1] = v.y;
        in[4 * q + 2] = v.z;
        in[4 * q + 3] = v.w;
      }
    }
    const uint32_t s_off = uint32_t(s0 - lane) * ROWB;    // staging offset of the lane's row at step s0+1
    const uint32_t xnext = x_s + uint32_t(s0 + U - lane);  // x of the lane's rows in the next block
    int32_t eq[4];
#pragma unroll
    for (int u = 0; u < U; ++u) {
      // lane 31's rows s0-30+u: quads of ring slots aligned at s0-30+4q (s0 - 28 = 0 mod 4)
      const uint32_t rout = ring_out + slot(s0 - 30 + (u & ~3)) + 4u * (u & 3);
      step<EDGE>(s0 + 1 + u, xc[u], in[u], s_off + uint32_t(u * ROWB), rout);
      asm volatile("ld.shared.u8 %0, [%1];" : "=r"(xc[u]) : "r"(xnext + uint32_t(u)));
      if constexpr (WF_NW8_DIRECT_EAST && WI == WARPS - 1) {
        // the band's east column, 4 rows per 16-byte store (rows s0-30+u-3 .. s0-30+u, an aligned
        // quad of the next band's / slab's global ring; rows <= 0 or > rows land in its slack,
        // which is never read)
        eq[u & 3] = east_last;
        if ((u & 3) == 3) {
          stg128_if(east_out, gout + (s0 - 33 + u), make_int4(eq[0], eq[1], eq[2], eq[3]));
          if (gx != nullptr) stg128_if(east_x, gx + (s0 - 33 + u), make_int4(eq[0], eq[1], eq[2], eq[3]));   // uniform
        }
      }
    }
  }

  // TMA store of rows r0 .. r0+31 (r0 >= 1) from the staging ring
  __device__ __forceinline__ void publish(int r0) {
    fence_proxy_async_smem();
    __syncwarp();
    if (lane == 0) {
      bulk_wait_read<1>();   // slots of the box issued two publishes ago may be rewritten next
      tma_store_2d(tmap, stage_s + uint32_t((r0 - 1) & (SR - 1)) * ROWB, ocol, r0 - 1);
      bulk_commit();
    }
    __syncwarp();
  }

  // end of the block s0+1 .. s0+U, then the CTA barrier.  When rows e-63 .. e-32 are complete
  // (lane 31 passed them) their 32-row box is stored: with WF_NW8_HELPER_TMA the warp only
  // fences its staged rows into the async proxy and the helper issues the TMA store after the
  // barrier (Helper::store_boxes); otherwise lane 0 issues it here.
  __device__ __forceinline__ void after_block(int s0) {
    const int e = s0 + U;   // last local step done
#if WF_NW8_HELPER_TMA
    if (e % 32 == 0 && e >= 64) fence_proxy_async_smem();   // the helper / storer warp stores the box
#else
    if (e % 32 == 0 && e >= 64) publish(e - 63);
#endif
    wf_jitter(1 + WI);
    cta_bar<NT>();
  }

  __device__ __forceinline__ void run() {
    const int Tw = rows + 31;                       // local steps of this warp
    const int Tc = Tw + (WARPS - 1) * LAG;          // CTA steps (every warp's blocks + the lags)
    const int Lw = WI * LAG;                        // this warp's lag in CTA steps
    // WF_TRACE=1 timeline, per band and warp (slots 8w..8w+7): [0] globaltimer at the band's
    // start, [1] when the warp starts its first block, [2] at the end of its sweep, [3] SM cycles
    // of the sweep
    unsigned long long* tr = (L.trace && lane == 0 && WI < 7) ? L.trace + size_t(band) * kTraceSlots + 8 * WI : nullptr;
    if (tr) tr[0] = globaltimer();
    cta_bar<NT>();   // the helper's prologue (row 1 and warp 0's first words) is in ring 0
    int B = 0;
    for (; B < Lw; B += U) cta_bar<NT>();   // before this warp's first block (its lag)
    // row 1's word (stored before this barrier) and the x codes of the first block
    if (is31) src = BOUND ? (LOCAL ? 0 : gap) : lds32(ring_in + slot(1));
    const long long c1 = clock64();
    if (tr) tr[1] = globaltimer();
    uint32_t xc[U];
    load_x(0, xc);
    int s0 = 0;   // local steps s0+1 .. s0+U of the block starting at CTA step B = s0 + Lw
    if constexpr (!LOCAL) {
      // NW: the ramp-up runs through the virtual rows (constructor) and the drain's rows > rows
      // are clipped by the tensor bounds and never read, so every block is a steady block
#pragma unroll 1
      for (; s0 < Tw; s0 += U) {
        block<false>(s0, xc);
        after_block(s0);
      }
    } else {
      // SW: ramp-up (lane 31 not yet on row 1) and steady blocks, then the drain
      for (; s0 < 31 && s0 < Tw; s0 += U) {
        block<true>(s0, xc);
        after_block(s0);
      }
#pragma unroll 1
      for (; s0 + U <= rows; s0 += U) {
        block<false>(s0, xc);
        after_block(s0);
      }
      for (; s0 < Tw; s0 += U) {
        block<true>(s0, xc);
        after_block(s0);
      }
    }
    for (B = s0 + Lw; B < Tc; B += U) cta_bar<NT>();   // the other warps' drain
    // the rows not yet stored: from the last published box on (s0 = ceil(Tw / U) * U)
    for (int r0 = s0 >= 64 ? (s0 / 32) * 32 - 31 : 1; r0 <= rows; r0 += 32) publish(r0);
    if (lane == 0) bulk_wait_all();
    if (tr) {
      tr[2] = globaltimer();
      tr[3] = static_cast<unsigned long long>(clock64() - c1);
    }
    if constexpr (LOCAL) L.lane_best[(size_t(band) * WARPS + WI) * 32 + lane] = make_int2(best, best_row);
  }
};

// Out-of-line slow path of the helper's inbound words: spin on the global quad at g (rows
// r0..r0+3, those <= rows) until none is EMPTY; a watchdog expiry returns failed = 1.
struct Slow4 {
  int4 v;
  int failed;
};
__device__ __noinline__ Slow4 slow_quad(const SweepLaunch& L, const int32_t* g, int r0, int rows, bool mine) {
  Slow4 r{make_int4(0, 0, 0, 0), 0};
  Watchdog wd;
  wd.start();
  for (;;) {
    r.v = mine ? ldg128_sys(g) : make_int4(0, 0, 0, 0);
    const bool st = mine && quad_stale(r.v, r0, rows);
    if (__all_sync(FULL, !st)) return r;
    if (__any_sync(FULL, wd.expired(L))) {
      r.failed = 1;
      return r;
    }
  }
}

// ---------------------------------------------------------------------------------------------
// The helper warp (warp WARPS): all global-memory hand-off traffic of the band.  It runs the
// CTA's block clock (one barrier per block) and, in CTA block j,
//   inbound  (band > 0 or slab > 0): writes the west words of warp 0's block j+1 -- rows
//            (j+1)U+2 .. (j+2)U+1, loaded DPRE blocks earlier -- into shared ring 0 after checking
//            them, resets their global slots, and loads the words of block j+1+DPRE;
//   outbound (a next band / slab exists): forwards the east words the last compute warp stored
//            into ring WARPS during block j-1 to the next band's / slab's global ring.
// Lane q < U/4 handles quad q (rows r0+4q .. r0+4q+3) of a block.
// ---------------------------------------------------------------------------------------------
template <int K, int WARPS, bool LOCAL, int U>
struct Helper {
  using S = Smem<K, WARPS>;
  static constexpr int LAG = 32 + U;
  static constexpr int NT = (WARPS + kExtraWarps) * 32;

  const SweepLaunch& L;
  const CUtensorMap* tmap;
  const int band, lane;
  int rows;
  bool inbound, outbound, mine;
  uint32_t ring0, ringW;
  uint32_t stage0;        // shared address of compute warp 0's staging ring
  int elast;              // every compute warp's last local block end (ceil(Tw / U) U)
  int32_t* gin;
  int32_t* gout;
  int4 emptyq;
  static constexpr int DP = WF_NW8_DPRE_ROWS / U > 0 ? WF_NW8_DPRE_ROWS / U : 1;   // blocks of lead
  int4 pre[DP];       // inbound quads of the next DP blocks (pre[0] = the next to deliver)
  bool failed = false;
  unsigned nslow = 0;     // WF_TRACE: blocks whose inbound quads were not all there when delivered
  Watchdog wd;

  __device__ __forceinline__ Helper(const SweepLaunch& L_, const CUtensorMap* tm, const CUtensorMap* tm_halo, const S& sm,
                                    int band_, int lane_, bool first)
      : L(L_), tmap(band_ < L_.halo_bands ? tm_halo : tm), band(band_), lane(lane_) {
    rows = L.rows;
    stage0 = saddr(sm.stage);
    elast = ((rows + 31 + U - 1) / U) * U;
    mine = lane < U / 4;
    ring0 = saddr(sm.ring);
    ringW = saddr(sm.ring) + uint32_t(WARPS) * RR * 4;
    const size_t es = gring_stride(rows);
    int32_t* gbase = reinterpret_cast<int32_t*>(L.edge);
    gin = gbase + size_t(band) * es + kGOff;
    gout = (band + 1 < L.nbands) ? gbase + size_t(band + 1) * es + kGOff
                                 : (L.next_edge ? reinterpret_cast<int32_t*>(L.next_edge) + kGOff : nullptr);
    inbound = !first;
    outbound = gout != nullptr;
    const int32_t e = lds32(saddr(sm.ctl + 31));   // EMPTY, written by the kernel prologue (opaque to ptxas)
    emptyq = make_int4(e, e, e, e);
#pragma unroll
    for (int i = 0; i < DP; ++i) pre[i] = make_int4(0, 0, 0, 0);
  }

  // inbound quad of lane q for the block of warp 0 starting at local step s0 (rows s0+2+4q ..)
  __device__ __forceinline__ int rq(int s0) const { return s0 + 2 + 4 * lane; }
  __device__ __forceinline__ int4 load_quad(int s0) const {
    const int r = rq(s0);
    return (mine && r <= rows) ? ldg128_sys(gin + r) : emptyq;
  }
  // check the quad of block s0 loaded DP blocks ago (pre[0]), spin if stale, store it into ring 0,
  // reset its global slots; then shift the queue and load block s0 + DP U
  __device__ __forceinline__ void deliver(int s0) {
    const int r = rq(s0);
    const bool need = mine && r <= rows;
    int4 v = pre[0];
    const bool st = need && quad_stale(v, r, rows);
    if (!failed && __any_sync(FULL, st)) {
      ++nslow;
      const Slow4 w = slow_quad(L, gin + r, r, rows, need);
      failed = w.failed != 0;
      if (need) v = w.v;
    }
    if (mine) sts128(ring0 + slot(r), v);
    if (need) stg128_sys(gin + r, emptyq);   // consumed: reset for the next run
#pragma unroll
    for (int i = 0; i + 1 < DP; ++i) pre[i] = pre[i + 1];
    pre[DP - 1] = load_quad(s0 + DP * U);
  }
  // forward the east words the last compute warp stored during its block s0 (rows s0-30 ..)
  __device__ __forceinline__ void forward(int s0) {
    const int r = s0 - 30 + 4 * lane;
    if (mine && r + 3 >= 1 && r <= rows) {
      const int4 v = lds128(ringW + slot(r));
      stg128_sys(gout + r, v);   // rows <= 0 / > rows land in the ring's slack (never read)
    }
  }

  // TMA stores of the 32-row boxes the compute warps completed at CTA step B (warp w's local
  // step e = B - w LAG, e = 0 mod 32, 64 <= e <= its last block end), one commit group per
  // call; the box of e is read out of its staging slots before the barrier at CTA step
  // B + 64, after which warp w may rewrite them (hence wait_group.read 3 with one group per
  // block).  Lane 0 only: bulk async-groups are per thread.
  __device__ __forceinline__ void store_boxes(int B) {
    if (lane != 0) return;
#pragma unroll
    for (int w = 0; w < WARPS; ++w) {
      const int e = B - w * LAG;
      if (e >= 64 && (e & 31) == 0 && e <= elast) {
        const int r0 = e - 63;
        tma_store_2d(tmap, stage0 + uint32_t(w) * SR * S::ROWB + uint32_t((r0 - 1) & (SR - 1)) * S::ROWB,
                     (band < L.halo_bands ? band : band - L.halo_bands) * L.band_w + w * 32 * K, r0 - 1);
      }
    }
    bulk_commit();
    bulk_wait_read<3>();
  }

  // the storer warp (WF_NW8_HELPER_TMA == 2): the CTA's barrier sequence with only the stores
  __device__ __forceinline__ void run_storer() {
    const int Tc = rows + 31 + (WARPS - 1) * LAG;
    cta_bar<NT>();
    int B = 0;
    for (; B < Tc; B += U) {
      wf_jitter(10);
      store_boxes(B);
      cta_bar<NT>();
    }
    store_boxes(B);
    if (lane == 0) bulk_wait_all();
  }

  __device__ __forceinline__ void run() {
    const int Tw = rows + 31;
    const int Tc = Tw + (WARPS - 1) * LAG;
    const int Ll = (WARPS - 1) * LAG;   // the last compute warp's lag
    if (band == L.export_band && L.next_edge && L.ack_self) {
      // the next slab must have drained (and reset) this ring in the previous run
      wd.start();
      for (;;) {
        const unsigned a = ld_relaxed_sys_u32(L.ack_self);
        if (__all_sync(FULL, static_cast<int>(a - (L.epoch - 1u)) >= 0)) break;
        if (__any_sync(FULL, wd.expired(L))) {
          failed = true;
          break;
        }
        __nanosleep(64);
      }
    }
    if (inbound) {
      // prologue: row 1 (lane 0 spins on it) and warp 0's first block, then preload block 1
      if (!failed) {
        wd.start();
        for (;;) {
          const int32_t v = lane == 0 ? ldg32_sys(gin + 1) : 0;
          if (__all_sync(FULL, lane != 0 || v != EMPTY)) {
            if (lane == 0) {
              sts32_if(true, ring0 + slot(1), v);
              stg32_sys(gin + 1, emptyq.x);   // consumed: reset for the next run
            }
            break;
          }
          if (__any_sync(FULL, wd.expired(L))) {
            failed = true;
            break;
          }
          __nanosleep(32);
        }
      }
#pragma unroll
      for (int i = 0; i < DP; ++i) pre[i] = load_quad(i * U);
      deliver(0);
    }
    cta_bar<NT>();   // warp 0's first block reads what the prologue stored
    int B = 0;
    for (; B < Tc; B += U) {
      // B = CTA step of this block's start; warp 0's current block has local start s0 = B
      wf_jitter(9);
      if (inbound && B + U < Tw) deliver(B + U);   // warp 0's next block starts at local step B + U
      if (!WF_NW8_DIRECT_EAST && outbound && B >= U) {   // the last warp's block that ended at this block's start
        const int s0 = B - U - Ll;
        if (s0 >= 0 && s0 < Tw) forward(s0);
      }
#if WF_NW8_HELPER_TMA == 1
      store_boxes(B);
#endif
      cta_bar<NT>();
    }
    if (!WF_NW8_DIRECT_EAST && outbound) {
      const int s0 = ((Tc + U - 1) / U) * U - U - Ll;   // the last warp's final block
      if (s0 >= 0 && s0 < Tw) forward(s0);
    }
#if WF_NW8_HELPER_TMA == 1
    store_boxes(B);   // boxes completed by the final block (the compute warps store the rest)
    if (lane == 0) bulk_wait_all();
#endif
    if (L.trace && lane == 0) L.trace[size_t(band) * kTraceSlots + 8 * WARPS + 4] = nslow;   // helper slot
    if (inbound && band == 0 && !L.first_slab && L.ack_prev) {   // predecessor slab may reuse this ring
      __threadfence_system();
      if (lane == 0) st_relaxed_sys_u32(L.ack_prev, L.epoch);
    }
  }
};

template <int K, int WARPS, int WI, bool LOCAL, int U>
__device__ __forceinline__ void dispatch(const SweepLaunch& L, const CUtensorMap* tm, const CUtensorMap* tmh,
                                         const Smem<K, WARPS>& sm, int band, int warp, int lane, bool first) {
  if constexpr (WI < WARPS) {
    if (warp == WI) {
      if constexpr (WI == 0) {
        if (first) {
          Warp<K, WARPS, 0, true, LOCAL, U> w(L, tm, tmh, sm, band, lane);
          w.run();
          return;
        }
      }
      Warp<K, WARPS, WI, false, LOCAL, U> w(L, tm, tmh, sm, band, lane);
      w.run();
    } else {
      dispatch<K, WARPS, WI + 1, LOCAL, U>(L, tm, tmh, sm, band, warp, lane, first);
    }
  } else {
    Helper<K, WARPS, LOCAL, U> h(L, tm, tmh, sm, band, lane, first);
    if (WF_NW8_HELPER_TMA == 2 && warp == WARPS + 1) h.run_storer();
    else h.run();
  }
}

template <int K, int WARPS, bool LOCAL, int U>
__global__ void __launch_bounds__((WARPS + kExtraWarps) * 32, 1)
    nw8_kernel(const __grid_constant__ SweepLaunch L, const __grid_constant__ CUtensorMap tmap,
               const __grid_constant__ CUtensorMap tmap_halo) {
  using S = Smem<K, WARPS>;
  extern __shared__ __align__(16) unsigned char nw8_smem_raw[];
  const S sm(nw8_smem_raw);
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  // shared x copy (row codes), once per CTA: x[r-1] for r = 1..rows
  {
    const uint8_t* x = static_cast<const uint8_t*>(L.row_in);
    const int n = L.rows;
    if ((reinterpret_cast<uintptr_t>(x) & 15u) == 0) {
      const int n16 = n >> 4;
      for (int i = threadIdx.x; i < n16; i += blockDim.x)
        reinterpret_cast<uint4*>(sm.x)[i] = __ldg(reinterpret_cast<const uint4*>(x) + i);
      for (int i = (n16 << 4) + threadIdx.x; i < n; i += blockDim.x) sm.x[i] = __ldg(x + i);
    } else {
      for (int i = threadIdx.x; i < n; i += blockDim.x) sm.x[i] = __ldg(x + i);
    }
    if (threadIdx.x == 0) sm.ctl[31] = EMPTY;
  }
  for (int band = blockIdx.x; band < L.nbands; band += gridDim.x) {
    __syncthreads();
    dispatch<K, WARPS, 0, LOCAL, U>(L, &tmap, &tmap_halo, sm, band, warp, lane, L.first_slab && band == 0);
    __syncthreads();
    if (run_failed(L)) return;
  }
}

constexpr int kU = WF_NW8_U;   // steps per lockstep block

template <int K, int WARPS, int U>
cudaError_t launch(const SweepLaunch& L, cudaStream_t s, size_t smem) {
  CUtensorMap tmap, tmap_halo;
  cudaError_t e = encode_plane_map(&tmap, L, 32 * K, 32);
  if (e != cudaSuccess) return e;
  tmap_halo = tmap;
  if (L.halo_bands > 0) {   // NEXT-4 overlap bands: their own scratch plane
    e = encode_map_2d(&tmap_halo, L.halo_out, int(L.halo_pitch), L.rows, L.halo_pitch, 32 * K, 32);
    if (e != cudaSuccess) return e;
  }
  auto kfn = L.local ? nw8_kernel<K, WARPS, true, U> : nw8_kernel<K, WARPS, false, U>;
  e = cudaFuncSetAttribute(kfn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  kfn<<<L.grid, (WARPS + kExtraWarps) * 32, smem, s>>>(L, tmap, tmap_halo);
  return cudaGetLastError();
}

// U = the strip (wf_params.strip): rows per lockstep block, per band-to-band / slab-to-slab
// hand-off and per helper message
template <int K, int WARPS, bool LOCAL, int U = kU>
Variant make() {
  return Variant{WF_FN_SEQCMP, LOCAL ? 1 : 0, K, WARPS, 1, (WARPS + kExtraWarps) * 32, Smem<K, WARPS>::bytes,
                 reinterpret_cast<const void*>(nw8_kernel<K, WARPS, LOCAL, U>), &launch<K, WARPS, U>, 8, {}, U};
}

}  // namespace nw8

// Both the global (local = 0) and the Smith-Waterman (local = 1, looked up with dsize = 1)
// variants; each entry's kernel pointer is the exact instantiation launch() uses.  The first
// entry of a (K, warps, local) is its default strip (kU); the strip axis (8 / 32 rows) is
// compiled for the two main tilings.
const Variant* nw8_table(size_t* n) {
  static const Variant v[] = {
      nw8::make<2, 4, false>(),     nw8::make<2, 2, false>(),     nw8::make<1, 4, false>(),
      nw8::make<1, 8, false>(),     nw8::make<4, 2, false>(),     nw8::make<4, 1, false>(),
      nw8::make<2, 1, false>(),     nw8::make<2, 4, true>(),      nw8::make<2, 2, true>(),
      nw8::make<1, 4, true>(),      nw8::make<4, 2, true>(),      nw8::make<2, 4, false, 8>(),
      nw8::make<2, 4, false, 32>(), nw8::make<4, 2, false, 8>(),  nw8::make<4, 2, false, 32>(),
  };
  *n = sizeof(v) / sizeof(v[0]);
  return v;
}

}  // namespace wfk
