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
//  * WARPS compute warps per CTA (4 = one per SM sub-partition), K = 2, no helper warps: the
//    row codes are copied to shared memory once per CTA and every warp feeds itself.
//  * Lane -> lane: SHFL.IDX rotation.  Lane 31's slot carries lane 0's NEXT west input, so the
//    only instructions on the lane-to-lane chain are SHFL and ONE VIADDMNMX:
//    E = max(W + K g, P_{K-1}) = H_{K-1} for lanes 0..30, max(W - 2^29, in) = in for lane 31.
//  * Warp -> warp inside a CTA: LOCKSTEP.  The warps of a CTA advance in blocks of U steps
//    separated by one named CTA barrier, warp w running LAG = 32 + U rows behind warp w-1.
//    Lane 31 of warp w-1 stores its east value of row r into a shared ring (plain int32, one
//    STS per step); by the lag, every word warp w needs in a block was stored before the
//    barrier that opens the block, so the reader loads U rows with U/4 broadcast 16-byte loads
//    and needs no flag, tag, sentinel or flow control (the barrier orders shared memory).
//  * Band -> band (CTA -> CTA) and slab -> slab (GPU -> GPU over NVLink): lane 31 of the last
//    warp stores the same words with st.relaxed.sys into the next band's / next slab's global
//    ring (slot r = row r; a peer / IPC address at the slab edge).  The consumer (warp 0 of
//    the next band) prefetches them PF blocks ahead with cp.async into a private shared ring,
//    checks that none is the EMPTY sentinel (one vote per block; a stale block spins on the
//    global words) and resets the global slots to EMPTY for the next run (between slabs the
//    reset is fenced before the per-run ack the producer waits on).
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

namespace nw8 {

constexpr int RR = 64;         // slots per shared warp -> warp ring (power of 2, > 2U)
constexpr int RG = 128;        // slots of warp 0's private prefetch ring (power of 2, >= (PF + 2) U)
constexpr int SR = 128;        // staging rows per warp (power of 2, = 4 TMA boxes)
constexpr int XPAD = 64;       // bytes of padding around the shared x copy
constexpr int XMAX = 65536;    // rows the shared x copy holds (ABI maximum 65535)
constexpr unsigned FULL = 0xffffffffu;
#ifndef WF_NW8_SEL
#define WF_NW8_SEL 0   // 1: lane 31's rotation slot by SEL after H (A/B experiments; 0 = the E form)
#endif
#ifndef WF_NW8_U
#define WF_NW8_U 16    // steps per lockstep block (A/B: 8 and 4 slower, profiles/r02_nw8_ab.txt)
#endif
#ifndef WF_NW8_PF
#define WF_NW8_PF 2    // blocks of global west-word prefetch
#endif
constexpr int32_t EMPTY = static_cast<int32_t>(0x80808080u);   // memset(0x80) pattern; |H| < 2^24

enum : int { SRC_BOUND = 0, SRC_SMEM = 1, SRC_GLOB = 2 };
enum : int { DST_SMEM = 1, DST_GLOB = 2 };

// global ring of band b: int32 slots, row r at base[b * stride + kGOff + r]; 32+ slots of
// slack on each side so that ramp-up / drain rows never leave it; the stride is a multiple of
// 4 and kGOff = 2 mod 4, so rows r0 .. r0+3 with r0 = 2 mod 4 are one aligned 16-byte quad.
// Fits in the host's per-band allocation of (edge_stride + 64) u64 words.
constexpr int kGOff = 34;
__host__ __device__ inline size_t gring_stride(int rows) { return ((size_t(rows) + 5) & ~size_t(3)) + 64; }

template <int K, int WARPS>
struct Smem {
  static constexpr int ROWB = 32 * K * 4;   // bytes per staged row of one warp
  static constexpr size_t stage_bytes = size_t(WARPS) * SR * ROWB;
  static constexpr size_t ring_bytes = size_t(WARPS) * RR * 4 + RG * 4;
  static constexpr size_t x_bytes = XMAX + 2 * XPAD;
  static constexpr size_t ctl_bytes = 128;
  static constexpr size_t bytes = 1024 + stage_bytes + ring_bytes + x_bytes + ctl_bytes;
  unsigned char* stage;   // [WARPS][SR][32K] int32 (TMA source), 1024-byte aligned
  int32_t* ring;          // [WARPS][RR]: ring w = west words of warp w (w >= 1)
  int32_t* pre;           // [RG]: warp 0's private prefetch ring (global west source)
  unsigned char* x;       // x[r - 1] = code of row r, r = 1..rows (XPAD bytes of slack each side)
  int* ctl;               // ctl[31] = EMPTY (read back as a register value)
  __device__ __forceinline__ explicit Smem(unsigned char* raw) {
    const uint32_t a = static_cast<uint32_t>(__cvta_generic_to_shared(raw));
    unsigned char* base = raw + ((1024u - (a & 1023u)) & 1023u);
    stage = base;
    ring = reinterpret_cast<int32_t*>(base + stage_bytes);
    pre = ring + WARPS * RR;
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
__device__ __forceinline__ int32_t lds32(uint32_t a) {
  int32_t v;
  asm volatile("ld.volatile.shared.s32 %0, [%1];" : "=r"(v) : "r"(a) : "memory");
  return v;
}
// predicated stores: a divergent `if (lane == 31)` would wrap the following shuffles in a
// reconvergence sequence
__device__ __forceinline__ void sts32_if(bool p, uint32_t a, int32_t v) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q st.shared.s32 [%0], %1; }" ::"r"(a), "r"(v),
               "r"(static_cast<int>(p)));
}
__device__ __forceinline__ void stg32_sys_if(bool p, int32_t* a, int32_t v) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q st.relaxed.sys.global.s32 [%0], %1; }" ::"l"(a), "r"(v),
               "r"(static_cast<int>(p)));
}
__device__ __forceinline__ void stg128_if(bool p, int32_t* a, const int4& e) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %1, 0; @q st.volatile.global.v4.s32 [%0], {%2, %3, %4, %5}; }" ::"l"(a),
               "r"(static_cast<int>(p)), "r"(e.x), "r"(e.y), "r"(e.z), "r"(e.w)
               : "memory");
}
__device__ __forceinline__ void cp_async16_if(bool p, uint32_t dst, const void* src) {
  asm volatile("{ .reg .pred q; setp.ne.b32 q, %2, 0; @q cp.async.cg.shared.global [%0], [%1], 16; }" ::"r"(dst),
               "l"(src), "r"(static_cast<int>(p))
               : "memory");
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void cp_async_wait() {
  asm volatile("cp.async.wait_group %0;" ::"n"(N) : "memory");
}
template <int THREADS>
__device__ __forceinline__ void cta_bar() {
  if constexpr (THREADS > 32) asm volatile("bar.sync 1, %0;" ::"n"(THREADS) : "memory");
}

// Out-of-line slow path of a global west source: spin on the words of rows r0 .. r0+U-1
// (those <= rows) until none is EMPTY; a watchdog expiry returns failed = 1.  Every exit is
// warp-uniform, and the caller's state stays in registers.
template <int U>
struct SlowU {
  int32_t v[U];
  int failed;
};
template <int U>
__device__ __noinline__ SlowU<U> slow_glob(const SweepLaunch& L, const int32_t* g, int r0, int rows) {
  SlowU<U> r;
  r.failed = 0;
  Watchdog wd;
  wd.start();
  for (;;) {
    bool st = false;
#pragma unroll
    for (int q = 0; q < U / 4; ++q) {
      const int4 v = ldg128_sys(g + 4 * q);
      r.v[4 * q] = v.x;
      r.v[4 * q + 1] = v.y;
      r.v[4 * q + 2] = v.z;
      r.v[4 * q + 3] = v.w;
    }
#pragma unroll
    for (int u = 0; u < U; ++u) st |= (r.v[u] == EMPTY) && (r0 + u <= rows);
    if (__all_sync(FULL, !st)) return r;
    if (__any_sync(FULL, wd.expired(L))) {
      r.failed = 1;
      return r;
    }
    __nanosleep(32);
  }
}

// ---------------------------------------------------------------------------------------------
// One compute warp: warp index WI of the CTA.  SRC: where lane 0's west inputs come from; DST:
// where lane 31's east outputs go (DST_GLOB with a NULL ring = nowhere: the last band of the
// last slab).  U: steps per lockstep block; PF: blocks of global prefetch (SRC_GLOB).
// ---------------------------------------------------------------------------------------------
template <int K, int WARPS, int WI, int SRC, int DST, bool LOCAL, int U, int PF>
struct Warp {
  using S = Smem<K, WARPS>;
  static constexpr int ROWB = S::ROWB;
  static constexpr int LAG = 32 + U;   // rows between consecutive warps (lockstep)
  static_assert(U % 4 == 0 && 32 % U == 0, "block of U steps: multiple of 4, divides 32");
  static_assert(RR > 2 * U && RG >= (PF + 2) * U, "ring sizes");
  static_assert(SR * ROWB <= 65536, "staging slot arithmetic");

  const SweepLaunch& L;
  const CUtensorMap* tmap;
  const int band, lane;
  const bool is31;
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
  uint32_t ring_in;       // shared address of ring WI (SMEM source) or the private ring (GLOB)
  uint32_t ring_out;      // shared address of ring WI + 1
  uint32_t x_s;           // shared address of the x copy (x of row r at x_s + r - 1)
  int32_t* gin;           // SRC_GLOB: this band's inbound global ring (row r at gin[r])
  int32_t* gout;          // DST_GLOB: next band's / slab's inbound global ring (or NULL)
  int4 emptyq;            // EMPTY x 4 (global ring resets)
  bool east31;            // lane 31 of a warp whose east words go somewhere (DST_GLOB with a ring)
  int32_t best = 0, best_row = 0;   // LOCAL: best cell value of the lane and the first row reaching it
  bool failed = false;    // a wait hit the watchdog: finish without waiting (results unspecified)
  int nslow = 0;          // WF_TRACE: blocks that entered the slow path
  Watchdog wd;

  __device__ __forceinline__ Warp(const SweepLaunch& L_, const CUtensorMap* tm, const S& sm, int band_, int lane_)
      : L(L_), tmap(tm), band(band_), lane(lane_), is31(lane_ == 31) {
    rows = L.rows;
    gap = L.gap;
    mmatch = L.match;
    mmis = L.mismatch;
#pragma unroll
    for (int m = 0; m < K; ++m) gk[m] = (m + 1) * gap;
    gLx = is31 ? -(1 << 29) : K * gap;
    const uint8_t* y = static_cast<const uint8_t*>(L.col_in);
    wcol = band * L.band_w + WI * 32 * K;
    const int jb = L.c0 + wcol + lane * K;   // global 0-based first column of the lane
#pragma unroll
    for (int m = 0; m < K; ++m) {
      const bool vc = jb + m < L.c1;
      ycode[m] = vc ? static_cast<uint32_t>(__ldg(y + jb + m)) : 0x100u;   // never equal to a code
      N[m] = (vc && !LOCAL) ? (jb + m + 1) * gap : 0;                      // H[0][j] = j g (NW), 0 (SW)
    }
    NWc = (!LOCAL) ? jb * gap : 0;                                          // H[0][jb]
    src = 0;
    srcl = (lane + 31) & 31;
    stage_s = saddr(sm.stage) + uint32_t(WI) * SR * ROWB;
    lane_off = uint32_t(lane) * 4 * K;
    ring_in = SRC == SRC_GLOB ? saddr(sm.pre) : saddr(sm.ring) + uint32_t(WI) * RR * 4;
    ring_out = saddr(sm.ring) + uint32_t(WI + 1) * RR * 4;
    x_s = saddr(sm.x);
    {
      const int32_t e = lds32(saddr(sm.ctl + 31));   // EMPTY, written by the kernel prologue (opaque to ptxas)
      emptyq = make_int4(e, e, e, e);
    }
    const size_t es = gring_stride(rows);
    int32_t* gbase = reinterpret_cast<int32_t*>(L.edge);
    gin = gbase + size_t(band) * es + kGOff;
    gout = (band + 1 < L.nbands) ? gbase + size_t(band + 1) * es + kGOff
                                 : (L.next_edge ? reinterpret_cast<int32_t*>(L.next_edge) + kGOff : nullptr);
    east31 = is31 && (DST == DST_SMEM || gout != nullptr);
  }

  static __device__ __forceinline__ int32_t t1f(int32_t n, int32_t g, int32_t d) {
    if constexpr (LOCAL) return __viaddmax_s32_relu(n, g, d);   // max(n + g, d, 0)
    else return __viaddmax_s32(n, g, d);
  }
  // ring slot byte offset of row r: rows r0 .. r0+3 with r0 = 2 mod 4 are one aligned quad
  template <int N_>
  static __device__ __forceinline__ uint32_t slot(int r) { return uint32_t((r + 2) & (N_ - 1)) * 4; }

  // ---- west words of one block: rows r0 .. r0+U-1 (r0 = 2 mod 4) -----------------------------
  __device__ __forceinline__ void load_in(int r0, int32_t (&in)[U]) const {
    constexpr int N_ = SRC == SRC_GLOB ? RG : RR;
#pragma unroll
    for (int q = 0; q < U / 4; ++q) {
      const int4 v = lds128(ring_in + slot<N_>(r0 + 4 * q));
      in[4 * q] = v.x;
      in[4 * q + 1] = v.y;
      in[4 * q + 2] = v.z;
      in[4 * q + 3] = v.w;
    }
  }
  template <bool EDGE>
  __device__ __forceinline__ bool stale(int r0, const int32_t (&in)[U]) const {
    bool st = false;
#pragma unroll
    for (int u = 0; u < U; ++u) st |= (in[u] == EMPTY) && (!EDGE || r0 + u <= rows);
    return st;
  }
  // SRC_GLOB: prefetch rows r0..r0+U-1 into the private shared ring (lane 31, 16-byte copies)
  __device__ __forceinline__ void prefetch(int r0) const {
#pragma unroll
    for (int q = 0; q < U / 4; ++q)
      cp_async16_if(is31 && r0 + 4 * q <= rows, ring_in + slot<RG>(r0 + 4 * q), gin + r0 + 4 * q);
    cp_async_commit();
  }
  // the words of row 1 (before local step 1)
  __device__ __forceinline__ int32_t word1() {
    if constexpr (SRC == SRC_BOUND) {
      return LOCAL ? 0 : gap;
    } else if constexpr (SRC == SRC_SMEM) {
      return lds32(ring_in + slot<RR>(1));
    } else {
      wd.start();
      for (;;) {
        const int32_t v = ldg32_sys(gin + 1);
        if (__all_sync(FULL, v != EMPTY)) {
          stg32_sys_if(lane == 0, gin + 1, emptyq.x);   // consumed: reset for the next run
          return v;
        }
        if (__any_sync(FULL, wd.expired(L))) {
          failed = true;
          return v;
        }
        __nanosleep(32);
      }
    }
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
#if WF_NW8_SEL
#pragma unroll
    for (int m = 0; m < K; ++m) H[m] = __viaddmax_s32(W, gk[m], P[m]);
    src = is31 ? in_next : H[K - 1];   // (A/B form: SEL on the lane chain instead of E)
#else
    const int32_t Px = is31 ? in_next : P[K - 1];
    src = __viaddmax_s32(W, gLx, Px);   // lanes 0..30: H[K-1]; lane 31: lane 0's next west input
#pragma unroll
    for (int m = 0; m < K; ++m) H[m] = __viaddmax_s32(W, gk[m], P[m]);
#endif
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
    // east hand-off: lane 31's row is s - 31
    if constexpr (DST == DST_SMEM) sts32_if(east31 && active, rout, H[K - 1]);
    else stg32_sys_if(east31 && active, gout + (s - 31), H[K - 1]);
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
  // gin_words: SRC_GLOB only -- on entry the (validated) words of this block, on exit those of
  // the next block (loaded at the start of this block, checked at its end: the load latency
  // and the check hide behind the block's steps)
  template <bool EDGE>
  __device__ __forceinline__ void block(int s0, uint32_t (&xc)[U], int32_t (&gw)[U]) {
    int32_t in[U];
    int32_t nx[U];
    const int r0 = s0 + 2;   // rows of lane 31's next west inputs: r0 .. r0+U-1
    if constexpr (SRC == SRC_BOUND) {
#pragma unroll
      for (int u = 0; u < U; ++u) in[u] = LOCAL ? 0 : (r0 + u) * gap;
    } else if constexpr (SRC == SRC_SMEM) {
      load_in(r0, in);   // stored by warp WI-1 before the barrier (lag LAG)
    } else {
#pragma unroll
      for (int u = 0; u < U; ++u) in[u] = gw[u];
      prefetch(r0 + (PF + 1) * U);
      cp_async_wait<PF>();   // the group of the next block's rows (issued PF blocks ago) has landed
      __syncwarp();
      load_in(r0 + U, nx);
    }
    const uint32_t s_off = uint32_t(s0 - lane) * ROWB;   // staging offset of the lane's row at step s0+1
    const uint32_t xnext = x_s + uint32_t(s0 + U - lane);  // x of the lane's rows in the next block
#pragma unroll
    for (int u = 0; u < U; ++u) {
      // lane 31's rows s0-30+u: quads of ring slots aligned at s0-30+4q (s0 - 28 = 0 mod 4)
      const uint32_t rout = ring_out + slot<RR>(s0 - 30 + (u & ~3)) + 4u * (u & 3);
      step<EDGE>(s0 + 1 + u, xc[u], in[u], s_off + uint32_t(u * ROWB), rout);
      asm volatile("ld.shared.u8 %0, [%1];" : "=r"(xc[u]) : "r"(xnext + uint32_t(u)));
    }
    if constexpr (SRC == SRC_GLOB) {
      // this block's global slots are consumed: reset them for the next run; validate the next
      // block's words (the slow path spins on the global words; every exit is warp-uniform)
#pragma unroll
      for (int q = 0; q < U / 4; ++q) stg128_if(lane == 0 && r0 + 4 * q <= rows, gin + r0 + 4 * q, emptyq);
      if (!failed && !__all_sync(FULL, !stale<true>(r0 + U, nx))) {
        const SlowU<U> r = slow_glob<U>(L, gin + r0 + U, r0 + U, rows);
        failed = r.failed != 0;
#pragma unroll
        for (int u = 0; u < U; ++u) nx[u] = r.v[u];
        ++nslow;
      }
#pragma unroll
      for (int u = 0; u < U; ++u) gw[u] = nx[u];
    }
  }

  // TMA store of rows r0 .. r0+31 (r0 >= 1) from the staging ring
  __device__ __forceinline__ void publish(int r0) {
    fence_proxy_async_smem();
    __syncwarp();
    if (lane == 0) {
      bulk_wait_read<1>();   // slots of the box issued two publishes ago may be rewritten next
      tma_store_2d(tmap, stage_s + uint32_t((r0 - 1) & (SR - 1)) * ROWB, wcol, r0 - 1);
      bulk_commit();
    }
    __syncwarp();
  }

  // end of the block s0+1 .. s0+U: TMA store of a completed 32-row box, then the CTA barrier
  __device__ __forceinline__ void after_block(int s0) {
    const int e = s0 + U;   // last local step done
    if (e % 32 == 0 && e >= 64) publish(e - 63);   // rows e-63 .. e-32 complete (lane 31 passed them)
    cta_bar<WARPS * 32>();
  }

  __device__ __forceinline__ void run() {
    const int Tw = rows + 31;                       // local steps of this warp
    const int Tc = Tw + (WARPS - 1) * LAG;          // CTA steps (every warp's blocks + the lags)
    const int Lw = WI * LAG;                        // this warp's lag in CTA steps
    // WF_TRACE=1 timeline, per band and warp (slots 8w..8w+7): [0] globaltimer at the band's
    // start, [1] when the warp's row 1 arrived, [2] at the end of its sweep, [3] SM cycles from
    // row 1 to the end, [4] blocks that took the slow (stale) path, [5] row-1 wait cycles
    unsigned long long* tr = (L.trace && lane == 0 && WI < 8) ? L.trace + size_t(band) * kTraceSlots + 8 * WI : nullptr;
    if (tr) tr[0] = globaltimer();
    long long c0 = clock64(), c1 = c0;
    int32_t gw[U];   // SRC_GLOB: validated words of the current block
#pragma unroll
    for (int u = 0; u < U; ++u) gw[u] = 0;
    if constexpr (SRC == SRC_GLOB) {
      // prime: blocks 0 .. PF (rows 2 .. (PF + 1) U + 1); block 0's words straight from global
#pragma unroll
      for (int k = 1; k <= PF; ++k) prefetch(2 + k * U);
      const SlowU<U> r = slow_glob<U>(L, gin + 2, 2, rows);
      failed = failed || r.failed != 0;
#pragma unroll
      for (int u = 0; u < U; ++u) gw[u] = r.v[u];
    }
    if (DST == DST_GLOB && band + 1 >= L.nbands && L.next_edge && L.ack_self) {
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
    int B = 0;
    for (; B < Lw; B += U) cta_bar<WARPS * 32>();   // before this warp's first block (its lag)
    // row 1's word (stored before this barrier) and the x codes of the first block
    {
      const int32_t in1 = word1();
      src = is31 ? in1 : 0;
      c1 = clock64();
      if (tr) tr[1] = globaltimer();
    }
    uint32_t xc[U];
    load_x(0, xc);
    int s0 = 0;   // local steps s0+1 .. s0+U of the block starting at CTA step B = s0 + Lw
    // ramp-up (lane 31 not yet on row 1) and steady blocks, then the drain
    for (; s0 < 31 && s0 < Tw; s0 += U) {
      block<true>(s0, xc, gw);
      after_block(s0);
    }
#pragma unroll 1
    for (; s0 + U <= rows; s0 += U) {
      block<false>(s0, xc, gw);
      after_block(s0);
    }
    for (; s0 < Tw; s0 += U) {
      block<true>(s0, xc, gw);
      after_block(s0);
    }
    for (B = s0 + Lw; B < Tc; B += U) cta_bar<WARPS * 32>();   // the other warps' drain
    // the rows not yet stored: from the last published box on
    const int e_last = s0;   // = ceil(Tw / U) * U
    int r0 = e_last >= 64 ? (e_last / 32) * 32 - 31 : 1;
    for (; r0 <= rows; r0 += 32) publish(r0);
    if constexpr (SRC == SRC_GLOB) {
      cp_async_wait<0>();
      if (band == 0 && !L.first_slab && L.ack_prev) {   // predecessor slab may reuse (write) this ring
        __threadfence_system();
        if (lane == 0) st_relaxed_sys_u32(L.ack_prev, L.epoch);
      }
    }
    if (lane == 0) bulk_wait_all();
    if (tr) {
      tr[2] = globaltimer();
      tr[3] = static_cast<unsigned long long>(clock64() - c1);
      tr[4] = static_cast<unsigned long long>(nslow);
      tr[5] = static_cast<unsigned long long>(c1 - c0);
    }
    if constexpr (LOCAL) L.lane_best[(size_t(band) * WARPS + WI) * 32 + lane] = make_int2(best, best_row);
  }
};

template <int K, int WARPS, int WI, bool LOCAL, int U, int PF>
__device__ __forceinline__ void run_warp(const SweepLaunch& L, const CUtensorMap* tm, const Smem<K, WARPS>& sm, int band,
                                         int lane, bool first) {
  constexpr int DST = WI == WARPS - 1 ? DST_GLOB : DST_SMEM;
  if constexpr (WI == 0) {
    if (first) {
      Warp<K, WARPS, WI, SRC_BOUND, DST, LOCAL, U, PF> w(L, tm, sm, band, lane);
      w.run();
    } else {
      Warp<K, WARPS, WI, SRC_GLOB, DST, LOCAL, U, PF> w(L, tm, sm, band, lane);
      w.run();
    }
  } else {
    Warp<K, WARPS, WI, SRC_SMEM, DST, LOCAL, U, PF> w(L, tm, sm, band, lane);
    w.run();
  }
}

template <int K, int WARPS, int WI, bool LOCAL, int U, int PF>
__device__ __forceinline__ void dispatch(const SweepLaunch& L, const CUtensorMap* tm, const Smem<K, WARPS>& sm, int band,
                                         int warp, int lane, bool first) {
  if constexpr (WI < WARPS) {
    if (warp == WI) run_warp<K, WARPS, WI, LOCAL, U, PF>(L, tm, sm, band, lane, first);
    else dispatch<K, WARPS, WI + 1, LOCAL, U, PF>(L, tm, sm, band, warp, lane, first);
  }
}

template <int K, int WARPS, bool LOCAL, int U, int PF>
__global__ void __launch_bounds__(WARPS * 32, 1)
    nw8_kernel(const __grid_constant__ SweepLaunch L, const __grid_constant__ CUtensorMap tmap) {
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
    dispatch<K, WARPS, 0, LOCAL, U, PF>(L, &tmap, sm, band, warp, lane, L.first_slab && band == 0);
    __syncthreads();
    if (run_failed(L)) return;
  }
}

constexpr int kU = WF_NW8_U;    // steps per lockstep block
constexpr int kPF = WF_NW8_PF;  // blocks of global prefetch

template <int K, int WARPS>
cudaError_t launch(const SweepLaunch& L, cudaStream_t s, size_t smem) {
  CUtensorMap tmap;
  cudaError_t e = encode_plane_map(&tmap, L, 32 * K, 32);
  if (e != cudaSuccess) return e;
  auto kfn = L.local ? nw8_kernel<K, WARPS, true, kU, kPF> : nw8_kernel<K, WARPS, false, kU, kPF>;
  e = cudaFuncSetAttribute(kfn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  kfn<<<L.grid, WARPS * 32, smem, s>>>(L, tmap);
  return cudaGetLastError();
}

template <int K, int WARPS, bool LOCAL>
Variant make() {
  return Variant{WF_FN_SEQCMP, LOCAL ? 1 : 0, K, WARPS, 1, WARPS * 32, Smem<K, WARPS>::bytes,
                 reinterpret_cast<const void*>(nw8_kernel<K, WARPS, LOCAL, kU, kPF>), &launch<K, WARPS>, 8};
}

}  // namespace nw8

// Both the global (local = 0) and the Smith-Waterman (local = 1, looked up with dsize = 1)
// variants; each entry's kernel pointer is the exact instantiation launch() uses.
const Variant* nw8_table(size_t* n) {
  static const Variant v[] = {
      nw8::make<2, 4, false>(), nw8::make<2, 2, false>(), nw8::make<1, 4, false>(), nw8::make<1, 8, false>(),
      nw8::make<4, 2, false>(), nw8::make<4, 1, false>(), nw8::make<2, 1, false>(), nw8::make<2, 4, true>(),
      nw8::make<2, 2, true>(),  nw8::make<1, 4, true>(),  nw8::make<4, 2, true>(),
  };
  *n = sizeof(v) / sizeof(v[0]);
  return v;
}

}  // namespace wfk
