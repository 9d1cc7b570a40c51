// wf_api.cpp -- the C ABI of libwf (include/wf.h): parameter validation, the planner
// (bands, slabs, persistent grid), library-owned scratch, and the launch path.
//
// The planner replaces the paper's tunables (Table 2: cpu-tile, band,
// gpu-count, gpu-tile, halo) with the B200 sweep's: lane columns k, warps per CTA band,
// lane skew d, GPU (slab) count and transport (DESIGN.md §6 "what differs from the paper").
#include <cuda_runtime.h>

#include <cstdarg>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <new>
#include <string>

#include "../../include/wf.h"
#include "wf_internal.h"

namespace wfk {
int variant_count();
}

struct wf_ctx {
  wf_params p{};
  int rank = 0, world = 1, device = 0, share = 1;
  int nf = 1, nbound = 0;
  int c0 = 0, c1 = 0;
  int cc0 = 0, halo_bands = 0, export_band = 0;   // NEXT-4 halo (Plan)
  void* halo_out = nullptr;                // overlap bands' scratch plane (rows x halo_pitch int32)
  int64_t halo_pitch = 0;
  int k = 4, warps = 2, skew = 2, band_w = 256, nbands = 1;
  int grid = 1;
  int smem = 0;
  int impl = 0;
  int strip = 0;                           // rows per hand-off block of the variant that runs
  void* base = nullptr;                    // one allocation: [control block | edge rings] (IPC-exportable)
  unsigned* ack = nullptr;                 // control word written by the successor slab
  unsigned long long* edge = nullptr;      // nbands * rows * nf LL words (library-owned)
  size_t edge_bytes = 0;
  unsigned* ack_prev = nullptr;            // predecessor's control word (local / peer / IPC)
  void* prev_ipc_base = nullptr;
  unsigned long long* next_edge = nullptr; // next slab's band-0 ring (peer / IPC / local)
  void* next_ipc_base = nullptr;
  int* err = nullptr;                      // device error word
  int* err_host = nullptr;                 // pinned copy of the error word after each run (async D2H)
  uint64_t watchdog = 0;                   // effective per-wait budget (SM cycles)
  uint32_t reported = 0;                   // epoch whose device error was already returned
  unsigned long long* trace = nullptr;     // WF_TRACE=1 timeline buffer (diagnostics)
  int2* lane_best = nullptr;               // local = 1: per-lane (best value, first row)
  int32_t* best_out = nullptr;             // local = 1: the slab's best cell (value, row, col)
  uint32_t epoch = 0;
  cudaEvent_t ev0 = nullptr, ev1 = nullptr;
  cudaEvent_t ev2 = nullptr;               // after the error-word copy of the last run
  bool ran = false;
  bool staged = false;                     // transport NCCL, world > 1: host-staged slab edges
  void* stage = nullptr;                   // rank < world-1: this slab's outbound edge ring (staged)
  size_t stage_bytes = 0;                  // one slab-edge message (a band-0 ring image)
  std::string msg;
};

namespace {

thread_local std::string g_last_error;
constexpr size_t kCtrlBytes = 256;   // control block at the head of the IPC-exportable allocation

wf_status fail(wf_ctx* c, wf_status st, const char* fmt, ...) {
  char buf[512];
  va_list ap;
  va_start(ap, fmt);
  vsnprintf(buf, sizeof buf, fmt, ap);
  va_end(ap);
  if (c) c->msg = buf;
  else g_last_error = buf;
  return st;
}

wf_status cuda_fail(wf_ctx* c, cudaError_t e, const char* what) {
  cudaGetLastError();
  return fail(c, e == cudaErrorMemoryAllocation ? WF_ENOMEM : WF_ECUDA, "%s: %s", what, cudaGetErrorString(e));
}

struct Plan {
  int nf, nbound, k, warps, skew, band_w, c0, c1, nbands;
  int cc0, halo_bands, export_band;   // NEXT-4 halo: first computed column, overlap bands, exporting band
  int impl;   // kernel generation actually used (wf_params.kernel, or the default's)
  int strip;  // wf_params.strip (0 = the generation's default block)
  int match, mismatch, gap;
};

// Defaults until the autotune table says otherwise (tools/autotune.py).
void defaults(const wf_params& p, int* k, int* w, int* d, int* impl) {
  *impl = p.kernel;
  if (p.fn == WF_FN_SEQCMP) {
    // generation 8 (wf_nw8.cu): 4 compute warps of K = 2 columns per lane, one long lane
    // pipeline with per-row hand-offs; generation 4 keeps (4, 2)
    const bool g4 = p.kernel == 4;
    *k = p.lane_cols ? p.lane_cols : (g4 ? 4 : 2);
    *w = p.warps ? p.warps : (g4 ? 2 : 4);
    *d = p.skew ? p.skew : 1;
  } else if (p.fn == WF_FN_NASH) {
    // one warp per column: lane_cols and skew are fixed at 1; 2 columns per CTA measured
    // fastest on C3 (profiles/autotune_C3.json)
    *k = p.lane_cols ? p.lane_cols : 1;
    *w = p.warps ? p.warps : 2;
    *d = p.skew ? p.skew : 1;
  } else {
    // synthetic: one column per lane keeps the tsize-deep FMA chain per step short.  From the
    // B200 sweep (profiles/tuner_sweep.json, 27 instances x all variants): one compute warp per
    // CTA with wf_syn for light cells; when a cell carries much FP work (dsize >= 3 with
    // tsize >= 1000, or dsize >= 5 with tsize >= 100) the generic sweep with 2 (dsize 3) or
    // 4 (dsize >= 5) warps per CTA wins (e.g. C5d 154 vs 197 ms).
    // Exception, measured after the idle-warp padding of wf_syn (dsize >= 3): at dsize 5 with
    // tsize >= 1000 the one-warp wf_syn CTA is faster again (C5d 154.5 -> 130.3 ms; dim 4096
    // 38.5 -> 31.4 ms); at tsize 100 (32 vs 61 ms) and dsize 3 / 4 (116 / 131 vs 142 / 144 ms)
    // the generic sweep stays ahead (tools/gpu_ps.sh).
    const bool syn_pad_wins = p.dsize == 5 && p.tsize >= 1000;
    const bool heavy = !syn_pad_wins && ((p.dsize >= 3 && p.tsize >= 1000) || (p.dsize >= 5 && p.tsize >= 100));
    *k = p.lane_cols ? p.lane_cols : 1;
    *w = p.warps ? p.warps : (heavy ? (p.dsize >= 5 ? 4 : 2) : 1);
    *d = p.skew ? p.skew : 1;
    if (!p.kernel && heavy && !p.warps && !p.lane_cols) *impl = 4;
  }
}

wf_status validate(const wf_params* p, int rank, Plan* out, wf_ctx* c) {
  if (!p) return fail(c, WF_EINVAL, "params is NULL");
  const int rows = p->dim;
  const int cols = p->cols ? p->cols : p->dim;
  if (rows < 1 || rows > 65535) return fail(c, WF_EINVAL, "dim=%d out of range 1..65535", rows);
  if (cols < 1 || cols > 65535) return fail(c, WF_EINVAL, "cols=%d out of range 1..65535", cols);
  if (p->kernel != 0 && p->kernel != 4 && p->kernel != 7 && p->kernel != 8)
    return fail(c, WF_EINVAL, "kernel=%d must be 0 (default), 4, 7 or 8", p->kernel);
  if (p->fn == WF_FN_SEQCMP && p->kernel == 7)
    return fail(c, WF_EUNSUPPORTED, "kernel=7: SEQCMP has generations 4 and 8 (the per-row v7 kernel was retired, DESIGN.md §12)");
  for (int i = 0; i < 3; ++i)
    if (p->reserved[i]) return fail(c, WF_EINVAL, "reserved[%d] must be 0", i);
  if (p->halo < 0) return fail(c, WF_EINVAL, "halo=%d must be >= 0", p->halo);
  if (p->alphabet < 0 || p->alphabet > 8) return fail(c, WF_EINVAL, "alphabet=%d out of range 0..8", p->alphabet);
  if (p->alphabet != 0 && p->fn != WF_FN_SEQCMP) return fail(c, WF_EINVAL, "alphabet applies to SEQCMP only");
  if (p->ngpus < 0 || p->ngpus > 8) return fail(c, WF_EINVAL, "ngpus=%d out of range 1..8", p->ngpus);
  const int G = p->ngpus ? p->ngpus : 1;
  if (rank < 0 || rank >= G) return fail(c, WF_EINVAL, "rank=%d out of range for ngpus=%d", rank, G);
  if (p->transport > WF_TRANSPORT_NCCL) return fail(c, WF_EINVAL, "transport=%u unknown", p->transport);
  // strip = rows per hand-off block (the band-to-band and slab-to-slab message); selectable
  // for generation 8 among its compiled blocks, fixed (0) for the other generations
  if (p->strip < 0 || p->strip > 65535) return fail(c, WF_EINVAL, "strip=%d out of range 0..65535", p->strip);
  if (p->lane_cols < 0 || p->warps < 0 || p->skew < 0)
    return fail(c, WF_EINVAL, "lane_cols/warps/skew must be >= 0");
  Plan pl{};
  switch (p->fn) {
    case WF_FN_SEQCMP: {
      if (p->tsize != 0) return fail(c, WF_EINVAL, "tsize=%d must be 0 for SEQCMP", p->tsize);
      if (p->dsize != 0) return fail(c, WF_EINVAL, "dsize=%d must be 0 for SEQCMP", p->dsize);
      if (p->local != 0 && p->local != 1) return fail(c, WF_EINVAL, "local=%d must be 0 or 1", p->local);
      const bool def = p->match == 0 && p->mismatch == 0 && p->gap == 0;
      pl.match = def ? 1 : p->match;
      pl.mismatch = def ? -1 : p->mismatch;
      pl.gap = def ? -1 : p->gap;
      if (pl.match < -64 || pl.match > 64) return fail(c, WF_EINVAL, "match=%d out of [-64,64]", pl.match);
      if (pl.mismatch < -64 || pl.mismatch > 64) return fail(c, WF_EINVAL, "mismatch=%d out of [-64,64]", pl.mismatch);
      if (pl.gap < -64 || pl.gap > 64) return fail(c, WF_EINVAL, "gap=%d out of [-64,64]", pl.gap);
      pl.nf = 1;
      pl.nbound = 0;
      break;
    }
    case WF_FN_SYNTHETIC:
      if (p->tsize < 0 || p->tsize > 1000000) return fail(c, WF_EINVAL, "tsize=%d out of range 0..1000000", p->tsize);
      if (p->dsize < 0 || p->dsize > 8) return fail(c, WF_EINVAL, "dsize=%d out of range 0..8", p->dsize);
      if ((long long)rows * cols > 2147483647LL)   // i1 = i*j of the last cell must fit int32 (R14)
        return fail(c, WF_EINVAL, "rows*cols=%lld too large for the int32 i1 = i*j field", (long long)rows * cols);
      pl.nf = 2 + p->dsize;
      pl.nbound = p->dsize;
      break;
    case WF_FN_NASH:
      if (p->tsize < 1 || p->tsize > 64) return fail(c, WF_EINVAL, "tsize=%d (strategies) out of range 1..64", p->tsize);
      if (p->dsize != 4) return fail(c, WF_EINVAL, "dsize=%d must be 4 for NASH", p->dsize);
      pl.nf = 4;
      pl.nbound = 4;
      break;
    default:
      return fail(c, WF_EINVAL, "fn=%d unknown", p->fn);
  }
  defaults(*p, &pl.k, &pl.warps, &pl.skew, &pl.impl);
  pl.strip = p->strip;
  // small NW grids (at most 3 default bands): 2 compute warps of K = 4 with 8-row strips halve the
  // in-CTA warp hops that dominate a short sweep -- C1 (dim 512): 0.0558 vs 0.0623 ms; from
  // dim 1024 up the tilings are within 1 % and (2, 4) wins at C4 (profiles/autotune_C1.json)
  if (p->fn == WF_FN_SEQCMP && !p->local && !p->lane_cols && !p->warps && !p->skew && !p->strip &&
      (p->kernel == 0 || p->kernel == 8) && cols <= 768) {
    pl.k = 4;
    pl.warps = 2;
    pl.strip = 8;
  }
  if (pl.k != 1 && pl.k != 2 && pl.k != 4 && pl.k != 8) return fail(c, WF_EINVAL, "lane_cols=%d not in {1,2,4,8}", pl.k);
  if (pl.warps < 1 || pl.warps > 8) return fail(c, WF_EINVAL, "warps=%d out of range 1..8", pl.warps);
  if (pl.skew < 1 || pl.skew > 4) return fail(c, WF_EINVAL, "skew=%d out of range 1..4", pl.skew);
  // a default band width whose shared-memory rings do not fit (many planes) halves until it does
  while (!p->warps && pl.warps > 1 &&
         !wfk::variant_exists(p->fn, p->fn == WF_FN_SEQCMP ? p->local : p->dsize, pl.k, pl.warps, pl.skew, pl.impl,
                              pl.strip))
    pl.warps /= 2;
  if (!wfk::variant_exists(p->fn, p->fn == WF_FN_SEQCMP ? p->local : p->dsize, pl.k, pl.warps, pl.skew, pl.impl,
                           pl.strip))
    return fail(c, WF_EUNSUPPORTED, "no kernel variant for fn=%d dsize=%d lane_cols=%d warps=%d skew=%d strip=%d",
                p->fn, p->dsize, pl.k, pl.warps, pl.skew, pl.strip);
  pl.strip = wfk::variant_strip(p->fn, p->fn == WF_FN_SEQCMP ? p->local : p->dsize, pl.k, pl.warps, pl.skew, pl.impl,
                                pl.strip);
  pl.band_w = p->fn == WF_FN_NASH ? pl.warps : pl.warps * 32 * pl.k;   // NASH: one column per warp
  // slabs: every slab but the last is a whole number of bands (its east column is then
  // owned by the last lane of its last band); bands are dealt out as evenly as possible
  const long long B = (cols + pl.band_w - 1) / pl.band_w;
  const long long b0 = B * rank / G, b1 = B * (rank + 1) / G;
  pl.c0 = (int)(b0 * pl.band_w < cols ? b0 * pl.band_w : cols);
  pl.c1 = (int)(b1 * pl.band_w < cols ? b1 * pl.band_w : cols);
  if (pl.c1 <= pl.c0) return fail(c, WF_EINVAL, "ngpus=%d leaves slab %d empty (cols=%d, band=%d)", G, rank, cols, pl.band_w);
  pl.nbands = (pl.c1 - pl.c0 + pl.band_w - 1) / pl.band_w;
  pl.cc0 = pl.c0;
  pl.halo_bands = 0;
  pl.export_band = pl.nbands - 1;
  if (p->halo) {
    // NEXT-4: slab g > 0 recomputes m = halo / band_w whole bands west of its own; slab g < G-1
    // exports the east edge of its band nbands-1-m (the column slab g+1's overlap starts after)
    if (p->fn != WF_FN_SEQCMP || p->local || !(pl.impl == 0 || pl.impl == 8) || pl.skew != 1 ||
        wfk::variant_strip(p->fn, 0, pl.k, pl.warps, pl.skew, pl.impl, pl.strip) == 0)
      return fail(c, WF_EUNSUPPORTED, "halo: global SEQCMP with the generation-8 sweep only");
    if (G < 2) return fail(c, WF_EINVAL, "halo=%d needs ngpus > 1", p->halo);
    if (p->halo % pl.band_w) return fail(c, WF_EINVAL, "halo=%d must be a multiple of the band width %d", p->halo, pl.band_w);
    const int m = p->halo / pl.band_w;
    const int own = pl.nbands;
    if (own <= m)
      return fail(c, WF_EINVAL, "halo=%d: every slab needs more than %d bands (slab %d has %d)", p->halo, m, rank, own);
    if (rank > 0) {
      pl.cc0 = pl.c0 - p->halo;
      pl.halo_bands = m;
      pl.nbands = own + m;
    }
    pl.export_band = pl.nbands - 1 - m;
  }
  *out = pl;
  return WF_OK;
}

}  // namespace

extern "C" {

int32_t wf_abi_version(void) { return WF_ABI_VERSION; }

const char* wf_build_info(void) {
  static std::string s;
  if (s.empty()) {
    char b[256];
    snprintf(b, sizeof b, "libwf abi=%d arch=sm_100a variants=%d cuda=%d", WF_ABI_VERSION, wfk::variant_count(),
             CUDART_VERSION);
    s = b;
  }
  return s.c_str();
}

const char* wf_last_error(const wf_ctx* c) {
  if (c) return c->msg.c_str();
  return g_last_error.c_str();
}

wf_status wf_query(const wf_params* p, int32_t rank, wf_layout* out) {
  if (!out) return fail(nullptr, WF_EINVAL, "layout is NULL");
  Plan pl;
  wf_status st = validate(p, rank, &pl, nullptr);
  if (st != WF_OK) return st;
  memset(out, 0, sizeof *out);
  out->nplanes = pl.nf;
  for (int f = 0; f < pl.nf; ++f) {
    out->plane_bytes[f] = 4;
    out->plane_is_float[f] = (p->fn == WF_FN_SYNTHETIC && f >= 2) ? 1 : 0;
  }
  out->nbound = pl.nbound;
  out->col_begin = pl.c0;
  out->col_end = pl.c1;
  out->min_pitch = ((int64_t)(pl.c1 - pl.c0) + 3) / 4 * 4;
  out->bytes_out = out->min_pitch * p->dim * 4 * pl.nf;
  out->lane_cols = pl.k;
  out->warps = pl.warps;
  out->skew = pl.skew;
  out->band_cols = pl.band_w;
  out->nbands = pl.nbands;
  out->strip = pl.strip;
  return WF_OK;
}

wf_status wf_create(const wf_params* p, const wf_dist* dist, wf_ctx** out) {
  if (!out) return fail(nullptr, WF_EINVAL, "out is NULL");
  *out = nullptr;
  const int rank = dist ? dist->rank : 0;
  if (dist) {
    const int G = p && p->ngpus ? p->ngpus : 1;
    if (dist->world != G) return fail(nullptr, WF_EINVAL, "dist.world=%d != params.ngpus=%d", dist->world, G);
    if (dist->device_share < 0 || dist->device_share > 64)
      return fail(nullptr, WF_EINVAL, "dist.device_share=%d out of range", dist->device_share);
  } else if (p && p->ngpus > 1) {
    return fail(nullptr, WF_EINVAL, "ngpus=%d needs a wf_dist", p->ngpus);
  }
  Plan pl;
  wf_status st = validate(p, rank, &pl, nullptr);
  if (st != WF_OK) return st;

  wf_ctx* c = new (std::nothrow) wf_ctx();
  if (!c) return fail(nullptr, WF_ENOMEM, "host allocation failed");
  c->p = *p;
  c->rank = rank;
  c->world = dist ? dist->world : 1;
  c->share = dist && dist->device_share > 1 ? dist->device_share : 1;
  c->nf = pl.nf;
  c->nbound = pl.nbound;
  c->c0 = pl.c0;
  c->cc0 = pl.cc0;
  c->halo_bands = pl.halo_bands;
  c->export_band = pl.export_band;
  c->c1 = pl.c1;
  c->k = pl.k;
  c->warps = pl.warps;
  c->impl = pl.impl;
  c->strip = pl.strip;
  c->skew = pl.skew;
  c->band_w = pl.band_w;
  c->nbands = pl.nbands;
  c->p.match = pl.match;
  c->p.mismatch = pl.mismatch;
  c->p.gap = pl.gap;

  cudaError_t e;
  if (dist && dist->device >= 0) {
    e = cudaSetDevice(dist->device);
    if (e != cudaSuccess) {
      st = cuda_fail(nullptr, e, "cudaSetDevice");
      delete c;
      return st;
    }
  }
  e = cudaGetDevice(&c->device);
  if (e != cudaSuccess) {
    st = cuda_fail(nullptr, e, "cudaGetDevice");
    delete c;
    return st;
  }
  // persistent grid: every CTA must be co-resident (flags are spun on, never relaunched)
  wfk::SweepLaunch L{};
  L.fn = p->fn;
  L.dsize = p->dsize;
  L.local = p->fn == WF_FN_SEQCMP ? p->local : 0;
  L.impl = pl.impl;
  L.strip = pl.strip;
  L.k = pl.k;
  L.warps = pl.warps;
  L.skew = pl.skew;
  c->smem = wfk::smem_bytes(L);
  int sms = 0, optin = 0;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, c->device);
  cudaDeviceGetAttribute(&optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, c->device);
  if (c->smem < 0 || c->smem > optin) {
    fail(nullptr, WF_EUNSUPPORTED, "variant needs %d B shared memory (device max %d)", c->smem, optin);
    delete c;
    return WF_EUNSUPPORTED;
  }
  const int occ = wfk::occupancy(L, c->smem);
  if (occ < 1) {
    fail(nullptr, WF_EUNSUPPORTED, "kernel variant cannot be resident (occupancy 0)");
    delete c;
    return WF_EUNSUPPORTED;
  }
  int cap = occ * sms / c->share;
  if (cap < 1) cap = 1;
  c->grid = pl.nbands < cap ? pl.nbands : cap;
  if (p->max_ctas && (int)p->max_ctas < c->grid) c->grid = (int)p->max_ctas;
  if (c->grid < 1) c->grid = 1;

  // per band: the inbound LL ring (edge_stride rows) plus 32 slots of slack on each side (the
  // generation-8 ring is addressed at +32 so that ramp-up / drain rows never leave it)
  // synthetic rings hold row records padded to 4-word multiples (wf_syn.cu syn_ring_words)
  const int ring_words = p->fn == WF_FN_SYNTHETIC ? ((pl.nf + 3) & ~3) : pl.nf;
  c->edge_bytes = (size_t)pl.nbands * (wfk::edge_stride(p->dim) + 64) * ring_words * sizeof(unsigned long long);
  e = cudaMalloc(&c->base, kCtrlBytes + c->edge_bytes);
  // control block 0; edge rings 0x80 bytes: the generation-8 EMPTY word (0x80808080), and a tag
  // no epoch ever takes for the LL-word generations
  if (e == cudaSuccess) e = cudaMemset(c->base, 0, kCtrlBytes);
  if (e == cudaSuccess) e = cudaMemset(static_cast<char*>(c->base) + kCtrlBytes, 0x80, c->edge_bytes);
  if (e == cudaSuccess) {
    c->ack = static_cast<unsigned*>(c->base);
    c->edge = reinterpret_cast<unsigned long long*>(static_cast<char*>(c->base) + kCtrlBytes);
  }
  // transport NCCL: the last band stores its east edge into a local outbound ring (same layout as
  // a band-0 inbound ring) which the caller ships with send/recv (wf_edge_export / import)
  c->staged = p->transport == WF_TRANSPORT_NCCL && c->world > 1;
  c->stage_bytes = (wfk::edge_stride(p->dim) + 64) * ring_words * sizeof(unsigned long long);
  if (e == cudaSuccess && c->staged && c->rank < c->world - 1) {
    e = cudaMalloc(&c->stage, c->stage_bytes);
    if (e == cudaSuccess) e = cudaMemset(c->stage, 0x80, c->stage_bytes);
    if (e == cudaSuccess) c->next_edge = static_cast<unsigned long long*>(c->stage);
  }
  if (e == cudaSuccess && c->halo_bands > 0) {   // NEXT-4: the overlap bands' cells (discarded)
    c->halo_pitch = (int64_t)c->halo_bands * c->band_w;
    e = cudaMalloc(&c->halo_out, (size_t)c->halo_pitch * p->dim * sizeof(int32_t));
  }
  if (e == cudaSuccess) e = cudaMalloc(&c->err, sizeof(int));
  if (e == cudaSuccess) e = cudaMemset(c->err, 0, sizeof(int));
  if (e == cudaSuccess) e = cudaMallocHost(&c->err_host, sizeof(int));
  if (e == cudaSuccess) *c->err_host = 0;
  // Default watchdog: a dependency wait may legitimately last the pipeline fill up to the last
  // band -- about nbands x 64 rows of steps, each step costing ~(tsize + 3) x max(dsize, 1) x 8
  // cycles for the synthetic cell (~100 cycles otherwise) -- so the budget scales with it
  // (a fixed 2^32 timed out valid large-tsize runs).
  if (e == cudaSuccess) {
    if (p->watchdog_cycles) {
      c->watchdog = p->watchdog_cycles;
    } else {
      const double step = p->fn == WF_FN_SYNTHETIC ? 8.0 * (p->tsize + 3) * (p->dsize > 1 ? p->dsize : 1)
                          : p->fn == WF_FN_NASH  ? 64.0 * p->tsize * p->tsize
                                                 : 100.0;
      const double fill = (double)pl.nbands * c->world * 64.0 * step * 4.0;   // x4 margin
      const double lim = 9.0e18;
      c->watchdog = (uint64_t)(fill > (double)(1ull << 32) ? (fill < lim ? fill : lim) : (double)(1ull << 32));
    }
  }
  if (e == cudaSuccess && L.local) {   // Smith-Waterman best-cell reduction scratch
    e = cudaMalloc(&c->lane_best, (size_t)pl.nbands * pl.warps * 32 * sizeof(int2));
    if (e == cudaSuccess) e = cudaMalloc(&c->best_out, 4 * sizeof(int32_t));
    if (e == cudaSuccess) e = cudaMemset(c->best_out, 0, 4 * sizeof(int32_t));
  }
  if (e == cudaSuccess) e = cudaEventCreate(&c->ev0);
  if (e == cudaSuccess) e = cudaEventCreate(&c->ev1);
  if (e == cudaSuccess) e = cudaEventCreateWithFlags(&c->ev2, cudaEventDisableTiming);
  if (e == cudaSuccess) e = cudaDeviceSynchronize();
  if (e != cudaSuccess) {
    st = cuda_fail(nullptr, e, "wf_create scratch");
    wf_destroy(c);
    return st;
  }
  *out = c;
  return WF_OK;
}

wf_status wf_destroy(wf_ctx* c) {
  if (!c) return WF_OK;
  int prev = -1;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  if (c->ev2) cudaEventSynchronize(c->ev2);   // the last run and its error-word copy
  if (c->next_ipc_base) cudaIpcCloseMemHandle(c->next_ipc_base);
  if (c->prev_ipc_base) cudaIpcCloseMemHandle(c->prev_ipc_base);
  if (c->base) cudaFree(c->base);
  if (c->stage) cudaFree(c->stage);
  if (c->halo_out) cudaFree(c->halo_out);
  if (c->err) cudaFree(c->err);
  if (c->err_host) cudaFreeHost(c->err_host);
  if (c->lane_best) cudaFree(c->lane_best);
  if (c->best_out) cudaFree(c->best_out);
  if (c->trace) cudaFree(c->trace);
  if (c->ev0) cudaEventDestroy(c->ev0);
  if (c->ev1) cudaEventDestroy(c->ev1);
  if (c->ev2) cudaEventDestroy(c->ev2);
  if (prev >= 0) cudaSetDevice(prev);
  cudaGetLastError();
  delete c;
  return WF_OK;
}

wf_status wf_link_local(wf_ctx* prev, wf_ctx* next) {
  if (!prev || !next) return fail(prev, WF_EINVAL, "wf_link_local: NULL context");
  if (prev->staged || next->staged)
    return fail(prev, WF_ESTATE, "wf_link_local: transport NCCL slabs exchange edges with wf_edge_export / wf_edge_import");
  if (next->rank != prev->rank + 1 || next->world != prev->world)
    return fail(prev, WF_EINVAL, "wf_link_local: ranks %d -> %d are not consecutive slabs", prev->rank, next->rank);
  if (prev->nf != next->nf || prev->p.dim != next->p.dim || prev->p.fn != next->p.fn ||
      prev->p.cols != next->p.cols || prev->p.tsize != next->p.tsize || prev->p.dsize != next->p.dsize ||
      prev->p.local != next->p.local || prev->impl != next->impl || prev->k != next->k ||
      prev->warps != next->warps || prev->skew != next->skew || prev->strip != next->strip ||
      prev->p.halo != next->p.halo)
    return fail(prev, WF_EINVAL, "wf_link_local: contexts describe different problems or tunings");
  if (prev->c1 != next->c0)
    return fail(prev, WF_EINVAL, "wf_link_local: slab %d ends at column %d but slab %d starts at %d", prev->rank,
                prev->c1, next->rank, next->c0);
  // the slabs' per-run acks and rings are epoch-paired: both must be linked before their first run
  if (prev->epoch != next->epoch || prev->ran || next->ran)
    return fail(prev, WF_ESTATE, "wf_link_local: link slabs before their first wf_run (epochs %u / %u)", prev->epoch,
                next->epoch);
  if (prev->device != next->device) {
    int can = 0;
    cudaDeviceCanAccessPeer(&can, prev->device, next->device);
    if (!can) return fail(prev, WF_ECOMM, "device %d cannot access peer %d", prev->device, next->device);
    int cur = 0;
    cudaGetDevice(&cur);
    cudaSetDevice(prev->device);
    cudaError_t e = cudaDeviceEnablePeerAccess(next->device, 0);
    cudaSetDevice(cur);
    if (e != cudaSuccess && e != cudaErrorPeerAccessAlreadyEnabled) {
      cudaGetLastError();
      return fail(prev, WF_ECOMM, "cudaDeviceEnablePeerAccess(%d->%d): %s", prev->device, next->device,
                  cudaGetErrorString(e));
    }
    cudaGetLastError();
  }
  if (next->device != prev->device) {
    int cur = 0;
    cudaGetDevice(&cur);
    cudaSetDevice(next->device);
    cudaError_t e = cudaDeviceEnablePeerAccess(prev->device, 0);   // next writes prev's ack word
    cudaSetDevice(cur);
    if (e != cudaSuccess && e != cudaErrorPeerAccessAlreadyEnabled) {
      cudaGetLastError();
      return fail(prev, WF_ECOMM, "cudaDeviceEnablePeerAccess(%d->%d): %s", next->device, prev->device,
                  cudaGetErrorString(e));
    }
    cudaGetLastError();
  }
  prev->next_edge = next->edge;   // next slab's band-0 inbound ring
  next->ack_prev = prev->ack;     // next acknowledges each drained run into prev's control word
  return WF_OK;
}

wf_status wf_ipc_handle(wf_ctx* c, void* handle) {
  if (!c || !handle) return fail(c, WF_EINVAL, "wf_ipc_handle: NULL argument");
  cudaIpcMemHandle_t h;
  cudaError_t e = cudaIpcGetMemHandle(&h, c->base);
  if (e != cudaSuccess) {
    cudaGetLastError();
    return fail(c, WF_ECOMM, "cudaIpcGetMemHandle: %s", cudaGetErrorString(e));
  }
  static_assert(sizeof(h) == WF_IPC_HANDLE_BYTES, "IPC handle size");
  memcpy(handle, &h, sizeof h);
  return WF_OK;
}

static wf_status open_ipc(wf_ctx* c, const void* handle, void** out) {
  cudaIpcMemHandle_t h;
  memcpy(&h, handle, sizeof h);
  cudaError_t e = cudaIpcOpenMemHandle(out, h, cudaIpcMemLazyEnablePeerAccess);
  if (e != cudaSuccess) {
    cudaGetLastError();
    return fail(c, WF_ECOMM, "cudaIpcOpenMemHandle: %s", cudaGetErrorString(e));
  }
  return WF_OK;
}

wf_status wf_connect(wf_ctx* c, const void* prev_handle, const void* next_handle) {
  if (!c) return fail(c, WF_EINVAL, "wf_connect: NULL context");
  if (c->staged) return fail(c, WF_ESTATE, "wf_connect: transport NCCL slabs exchange edges with wf_edge_export / wf_edge_import");
  // the slabs' per-run acks and rings are epoch-paired: every rank connects before its first run
  // (all ranks then issue the same sequence of wf_run calls)
  if (c->ran || c->epoch != 0)
    return fail(c, WF_ESTATE, "wf_connect: connect before the first wf_run (this context already ran %u times)", c->epoch);
  if ((c->rank > 0) != (prev_handle != nullptr))
    return fail(c, WF_EINVAL, "wf_connect: rank %d %s a predecessor handle", c->rank, c->rank > 0 ? "needs" : "takes no");
  if ((c->rank < c->world - 1) != (next_handle != nullptr))
    return fail(c, WF_EINVAL, "wf_connect: rank %d %s a successor handle", c->rank,
                c->rank < c->world - 1 ? "needs" : "takes no");
  int cur = 0;
  cudaGetDevice(&cur);
  cudaSetDevice(c->device);
  wf_status st = WF_OK;
  if (next_handle) {
    void* p = nullptr;
    st = open_ipc(c, next_handle, &p);
    if (st == WF_OK) {
      c->next_ipc_base = p;
      c->next_edge = reinterpret_cast<unsigned long long*>(static_cast<char*>(p) + kCtrlBytes);
    }
  }
  if (st == WF_OK && prev_handle) {
    void* p = nullptr;
    st = open_ipc(c, prev_handle, &p);
    if (st == WF_OK) {
      c->prev_ipc_base = p;
      c->ack_prev = static_cast<unsigned*>(p);
    }
  }
  cudaSetDevice(cur);
  return st;
}

wf_status wf_run(wf_ctx* c, const wf_io* io, void* cuda_stream) {
  if (!c) return fail(nullptr, WF_EINVAL, "wf_run: NULL context");
  if (!io) return fail(c, WF_EINVAL, "wf_run: io is NULL");
  const wf_params& p = c->p;
  const int cols = p.cols ? p.cols : p.dim;
  if (c->world > 1 && c->rank < c->world - 1 && !c->next_edge)
    return fail(c, WF_ESTATE, "wf_run: slab %d is not linked to its successor (wf_link_local / wf_connect)", c->rank);
  if (!io->row_in || !io->col_in) return fail(c, WF_EINVAL, "wf_run: row_in/col_in must be device pointers");
  const int64_t min_pitch = ((int64_t)(c->c1 - c->c0) + 3) / 4 * 4;
  if (io->out_pitch < min_pitch || io->out_pitch % 4 != 0)
    return fail(c, WF_EINVAL, "wf_run: out_pitch=%lld must be a multiple of 4 and >= %lld", (long long)io->out_pitch,
                (long long)min_pitch);
  for (int f = 0; f < c->nf; ++f) {
    if (!io->out[f]) return fail(c, WF_EINVAL, "wf_run: out[%d] is NULL", f);
    if (reinterpret_cast<uintptr_t>(io->out[f]) % 16) return fail(c, WF_EINVAL, "wf_run: out[%d] not 16-byte aligned", f);
  }
  for (int b = 0; b < c->nbound; ++b)
    if (!io->top[b] || !io->left[b]) return fail(c, WF_EINVAL, "wf_run: top[%d]/left[%d] must be set", b, b);

  wfk::SweepLaunch L{};
  L.fn = p.fn;
  L.rows = p.dim;
  L.cols = cols;
  L.tsize = p.tsize;
  L.dsize = p.dsize;
  L.local = p.fn == WF_FN_SEQCMP ? p.local : 0;
  L.impl = c->impl;
  L.strip = c->strip;
  L.lane_best = c->lane_best;
  L.best_out = c->best_out;
  L.c0 = c->c0;
  L.c1 = c->c1;
  L.cc0 = c->cc0;
  L.halo_bands = c->halo_bands;
  L.export_band = c->export_band;
  L.halo_out = c->halo_out;
  L.halo_pitch = c->halo_pitch;
  L.match = p.match;
  L.mismatch = p.mismatch;
  L.gap = p.gap;
  L.alphabet = p.alphabet;
  L.k = c->k;
  L.warps = c->warps;
  L.skew = c->skew;
  L.band_w = c->band_w;
  L.nbands = c->nbands;
  L.grid = c->grid;
  L.row_in = io->row_in;
  L.col_in = io->col_in;
  for (int f = 0; f < WF_MAX_PLANES; ++f) {
    L.top[f] = io->top[f];
    L.left[f] = io->left[f];
    L.out[f] = io->out[f];
  }
  L.pitch = io->out_pitch;
  L.edge = c->edge;
  L.next_edge = c->next_edge;
  // staged slabs: the host orders each run's edge message after the producer and before the
  // consumer on the streams, so there is no cross-run ack between slabs
  L.ack_self = c->staged ? nullptr : c->ack;
  L.ack_prev = c->staged ? nullptr : c->ack_prev;
  L.first_slab = c->rank == 0;
  // a device error of the previous run that has already completed (its error word was copied to
  // pinned host memory behind it) is reported here, once, without blocking (include/wf.h)
  if (c->ran && c->reported != c->epoch && cudaEventQuery(c->ev2) == cudaSuccess) {
    const int w = *reinterpret_cast<volatile int*>(c->err_host);
    if (((unsigned)w >> 4) == (c->epoch & 0x0FFFFFFFu) && (w & 15) == wfk::DEV_TIMEOUT) {
      c->reported = c->epoch;
      return fail(c, WF_ETIMEOUT, "watchdog fired in the previous run (epoch %u; budget %llu cycles per wait)",
                  c->epoch, (unsigned long long)c->watchdog);
    }
  } else {
    cudaGetLastError();
  }
  L.epoch = ++c->epoch;
  if ((L.epoch & 0x0FFFFFFFu) == 0) L.epoch = ++c->epoch;   // tag 0 marks "never written"
  L.err = c->err;
  if (!c->trace && getenv("WF_TRACE") && getenv("WF_TRACE")[0] == '1') {
    cudaMalloc(&c->trace, (size_t)c->nbands * wfk::kTraceSlots * 8);
    cudaGetLastError();
  }
  if (c->trace) cudaMemsetAsync(c->trace, 0, (size_t)c->nbands * wfk::kTraceSlots * 8, static_cast<cudaStream_t>(cuda_stream));
  L.trace = c->trace;
  L.watchdog = c->watchdog;

  int prev = -1;
  cudaGetDevice(&prev);
  if (prev != c->device) cudaSetDevice(c->device);
  cudaStream_t s = static_cast<cudaStream_t>(cuda_stream);
  cudaError_t e = cudaEventRecord(c->ev0, s);
  if (e == cudaSuccess) e = wfk::launch(L, s);
  if (e == cudaSuccess && L.local) e = wfk::launch_sw_best(L, s);   // part of the step: inside the timed events
  if (e == cudaSuccess) e = cudaEventRecord(c->ev1, s);
  if (e == cudaSuccess) e = cudaMemcpyAsync(c->err_host, c->err, sizeof(int), cudaMemcpyDeviceToHost, s);
  if (e == cudaSuccess) e = cudaEventRecord(c->ev2, s);
  if (prev >= 0 && prev != c->device) cudaSetDevice(prev);
  if (e != cudaSuccess) return cuda_fail(c, e, "wf_run launch");
  c->ran = true;
  return WF_OK;
}

wf_status wf_sync(wf_ctx* c) {
  if (!c) return fail(nullptr, WF_EINVAL, "wf_sync: NULL context");
  if (!c->ran) return WF_OK;
  cudaError_t e = cudaEventSynchronize(c->ev1);
  if (e != cudaSuccess) return cuda_fail(c, e, "wf_sync");
  int w = 0;
  e = cudaMemcpy(&w, c->err, sizeof w, cudaMemcpyDeviceToHost);
  if (e != cudaSuccess) return cuda_fail(c, e, "wf_sync error word");
  if (((unsigned)w >> 4) == (c->epoch & 0x0FFFFFFFu) && (w & 15) == wfk::DEV_TIMEOUT) {
    c->reported = c->epoch;
    return fail(c, WF_ETIMEOUT,
                "watchdog: a dependency wait exceeded %llu cycles (run epoch %u; linked slabs must issue the same "
                "sequence of wf_run calls)",
                (unsigned long long)c->watchdog, c->epoch);
  }
  return WF_OK;
}

wf_status wf_edge_bytes(const wf_ctx* c, size_t* bytes) {
  if (!c || !bytes) return fail(nullptr, WF_EINVAL, "wf_edge_bytes: NULL argument");
  if (!c->staged) return fail(const_cast<wf_ctx*>(c), WF_ESTATE, "wf_edge_bytes: not a transport NCCL slab");
  *bytes = c->stage_bytes;
  return WF_OK;
}

static wf_status edge_copy(wf_ctx* c, void* dst, const void* src, void* stream, const char* what) {
  int prev = -1;
  cudaGetDevice(&prev);
  if (prev != c->device) cudaSetDevice(c->device);
  cudaError_t e = cudaMemcpyAsync(dst, src, c->stage_bytes, cudaMemcpyDefault, static_cast<cudaStream_t>(stream));
  if (prev >= 0 && prev != c->device) cudaSetDevice(prev);
  if (e != cudaSuccess) return cuda_fail(c, e, what);
  return WF_OK;
}

wf_status wf_edge_export(wf_ctx* c, void* dst, void* cuda_stream) {
  if (!c || !dst) return fail(c, WF_EINVAL, "wf_edge_export: NULL argument");
  if (!c->staged || c->rank >= c->world - 1)
    return fail(c, WF_ESTATE, "wf_edge_export: only a transport NCCL slab with a successor exports its edge");
  return edge_copy(c, dst, c->stage, cuda_stream, "wf_edge_export");
}

wf_status wf_edge_import(wf_ctx* c, const void* src, void* cuda_stream) {
  if (!c || !src) return fail(c, WF_EINVAL, "wf_edge_import: NULL argument");
  if (!c->staged || c->rank == 0)
    return fail(c, WF_ESTATE, "wf_edge_import: only a transport NCCL slab with a predecessor imports an edge");
  return edge_copy(c, c->edge, src, cuda_stream, "wf_edge_import");
}

wf_status wf_debug_trace(wf_ctx* c, void* host, size_t bytes, int32_t* slots_per_band) {
  if (!c || !host || !slots_per_band) return fail(c, WF_EINVAL, "wf_debug_trace: NULL argument");
  *slots_per_band = wfk::kTraceSlots;
  if (!c->trace) return fail(c, WF_ESTATE, "wf_debug_trace: run with WF_TRACE=1 in the environment");
  const size_t need = (size_t)c->nbands * wfk::kTraceSlots * 8;
  cudaError_t e = cudaMemcpy(host, c->trace, bytes < need ? bytes : need, cudaMemcpyDeviceToHost);
  if (e != cudaSuccess) return cuda_fail(c, e, "wf_debug_trace");
  return WF_OK;
}

wf_status wf_local_best(wf_ctx* c, int32_t* score, int32_t* row, int32_t* col) {
  if (!c || !score || !row || !col) return fail(c, WF_EINVAL, "wf_local_best: NULL argument");
  if (!(c->p.fn == WF_FN_SEQCMP && c->p.local == 1)) return fail(c, WF_ESTATE, "wf_local_best: context is not local SEQCMP");
  if (!c->ran) return fail(c, WF_ESTATE, "wf_local_best: no run yet");
  cudaError_t e = cudaEventSynchronize(c->ev1);
  int32_t h[4] = {0, 0, 0, 0};
  if (e == cudaSuccess) e = cudaMemcpy(h, c->best_out, sizeof h, cudaMemcpyDeviceToHost);
  if (e != cudaSuccess) return cuda_fail(c, e, "wf_local_best");
  *score = h[0];
  *row = h[1];
  *col = h[2];
  return WF_OK;
}

wf_status wf_last_run_ms(wf_ctx* c, float* ms) {
  if (!c || !ms) return fail(c, WF_EINVAL, "wf_last_run_ms: NULL argument");
  if (!c->ran) return fail(c, WF_ESTATE, "wf_last_run_ms: no run yet");
  cudaError_t e = cudaEventQuery(c->ev1);
  if (e == cudaErrorNotReady) return fail(c, WF_ESTATE, "wf_last_run_ms: run still in flight");
  if (e != cudaSuccess) return cuda_fail(c, e, "wf_last_run_ms");
  e = cudaEventElapsedTime(ms, c->ev0, c->ev1);
  if (e != cudaSuccess) return cuda_fail(c, e, "cudaEventElapsedTime");
  return WF_OK;
}

}  // extern "C"
