/*
 * wf.h -- C ABI of libwf, the B200 (sm_100a) wavefront sweep.
 *
 * The operation (Sec. 1, Fig. 1): a two-dimensional wavefront
 * "abstracts computations which evaluate a class of multidimensional recurrence
 * relations ... The values of the relation are computed into a multidimensional
 * array.  Computation starts at position (0,0) and propagates to neighboring
 * elements in a series of diagonal bands".  libwf evaluates
 *
 *     a[i][j] = f(a[i-1][j], a[i][j-1], a[i-1][j-1], x_i, y_j)     1 <= i <= rows, 1 <= j <= cols
 *
 * over a rows x cols interior whose row 0 and column 0 are the boundary
 * (reading R2), for the paper's three applications (P:349-375 synthetic,
 * P:428-431 Nash equilibrium, P:432-435 biological sequence comparison).  The
 * pattern's API "requires the programmer to code only application specific
 * aspects": the caller picks f by id and supplies the instance
 * features of Table 1 (dim, tsize, dsize).
 *
 * Every entry point returns a wf_status (0 = OK).  No C++ exception or longjmp
 * crosses this boundary.  Status codes are the ABI; messages are advisory.
 * Threading: a context is not thread-safe; distinct contexts are independent.
 * Determinism: the output is a pure function of (params, inputs); it does not
 * depend on tiling, skew, strip, slab count or transport.
 */
#ifndef WF_H
#define WF_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define WF_ABI_VERSION 1
#define WF_MAX_PLANES 10   /* 2 ints + 8 floats (synthetic, dsize <= 8) */
#define WF_IPC_HANDLE_BYTES 64

typedef enum {
  WF_OK = 0,
  WF_EINVAL = 1,          /* a parameter is out of range; message names the field */
  WF_ENOMEM = 2,          /* device or host allocation failed */
  WF_ECUDA = 3,           /* a CUDA runtime error (message carries the CUDA string) */
  WF_ECOMM = 4,           /* inter-GPU setup failed (peer access / IPC) */
  WF_ETIMEOUT = 5,        /* a dependency flag was not satisfied within the watchdog budget */
  WF_EUNSUPPORTED = 6,    /* valid but not built (e.g. a tuning combination without a kernel) */
  WF_ESTATE = 7           /* call not valid in the context's current state */
} wf_status;

/* Cell functions (the paper's applications). */
typedef enum {
  /* Synthetic application, PAPER.md P:349-375 (Sec. 3.1.1): element = 2 int32 + dsize fp32;
   * tsize = inner iteration count.  Planes: 0 = i0 (int32), 1 = i1 (int32), 2.. = f[d] (fp32).
   *   i0 = max(max(N.i0, NW.i0), W.i0) + 1;   i1 = ((N.i1 - NW.i1) + 1) + W.i1
   *   c = (u_i * v_j) * 2^-12;  x_d = ((N.f_d + NW.f_d) + W.f_d) * fl(1/3);
   *   tsize times: x_d = fma(x_d, 1 - 2^-12, c)            (readings R4-R6, R11)
   * Boundary: i0 = -1, i1 = 0; floats from top/left planes. */
  WF_FN_SYNTHETIC = 0,
  /* Nash-equilibrium stand-in, PAPER.md P:428-431, P:437-439 (dsize = 4):
   * element = 4 int32 (count of pure equilibria, first equilibrium index, its two payoffs)
   * of an n x n bimatrix game (n = tsize) whose payoffs hash the neighbours
   * (reading R8).  Kernel: one warp per column (lane_cols = skew = 1;
   * warps in {1, 2, 4, 8} = columns per band; default 8). */
  WF_FN_NASH = 1,
  /* Sequence comparison, PAPER.md P:432-435 ("Biological Sequence Comparison [2]"),
   * P:732 ("Smith-Waterman"); Needleman-Wunsch global alignment with linear gap:
   *   H[i][0] = i*gap, H[0][j] = j*gap,
   *   H[i][j] = max(H[i-1][j-1] + (x_i == y_j ? match : mismatch), H[i-1][j] + gap, H[i][j-1] + gap)
   * One int32 plane.  local = 1: Smith-Waterman local alignment, H[i][0] = H[0][j] = 0,
   *   H[i][j] = max(0, <the three terms above>); the run also reduces the first (row-major)
   *   cell holding the maximum, read with wf_local_best. */
  WF_FN_SEQCMP = 2
} wf_fn;

typedef enum { WF_TRANSPORT_P2P = 0, WF_TRANSPORT_NCCL = 1 } wf_transport;

typedef struct {
  int32_t dim;          /* Table 1 'dim': rows of the interior, 1..65535 */
  int32_t cols;         /* 0 = square (cols = dim); else 1..65535 ("could be lifted") */
  int32_t fn;           /* wf_fn */
  int32_t tsize;        /* Table 1 'tsize': SYNTHETIC trip count 0..1000000; NASH strategies n 1..64;
                           SEQCMP must be 0 */
  int32_t dsize;        /* Table 1 'dsize': SYNTHETIC 0..8 fp32 items; NASH must be 4; SEQCMP must be 0 */
  int32_t lane_cols;    /* tunable k: adjacent columns owned by one lane (1, 2, 4, 8); 0 = default */
  int32_t warps;        /* tunable: compute warps per CTA = column groups per band (1..8); 0 = default */
  int32_t skew;         /* tunable d: row lag between neighbouring lanes (1..4); 0 = default */
  int32_t strip;        /* tunable: rows per hand-off block -- the unit in which a band passes its east
                           column to the next band and a slab to the next slab (the paper's halo-swap
                           interval).  0 = default (16).  Generation 8
                           compiles 8 / 16 / 32 for its main tilings (wf_query reports the one that
                           runs); the other generations have a fixed block and need 0; other values
                           -> WF_EUNSUPPORTED */
  int32_t ngpus;        /* slabs (column blocks), 1..8; see wf_dist */
  int32_t match, mismatch, gap;  /* SEQCMP scores, each in [-64, 64]; defaults used if all three 0 */
  int32_t local;        /* SEQCMP: 0 = global (Needleman-Wunsch), 1 = local (Smith-Waterman) */
  uint32_t transport;   /* wf_transport for ngpus > 1:
                           P2P (default) = the sweep stores the slab's east edge straight into the
                           successor's ring (wf_link_local / wf_connect), pipelined row block by row block;
                           NCCL = the host-staged fallback for systems without peer access: each slab
                           writes its east edge into a library buffer, the caller moves it with the
                           process group's send/recv (wf_edge_export / wf_edge_import) and slab g+1 runs
                           after slab g -- the paper's host-staged halo swap, not pipelined */
  uint32_t max_ctas;    /* 0 = all resident CTAs; else an upper bound (tests of the band loop) */
  uint64_t watchdog_cycles; /* spin budget per dependency wait (SM clock cycles); 0 = default: the larger of
                               2^32 and 4x the expected pipeline fill (bands x slabs x 64 rows x the
                               per-step cell cost estimate of fn / tsize / dsize) */
  int32_t alphabet;     /* SEQCMP: 0 = residue codes may be any byte value; 1..8 = every code in
                           row_in/col_in is < alphabet (e.g. 4 for DNA) -- enables the byte-permute
                           score lookup; codes outside the promise give unspecified scores */
  int32_t kernel;       /* kernel generation: 0 = the library's default for the function (tuned, DESIGN.md
                           §7).  SEQCMP: 8 = the lockstep lane pipeline (wf_nw8.cu; the default where its
                           (lane_cols, warps) is compiled, skew 1), 4 = the block hand-off sweep (wf_nw.cuh;
                           every other tuning).  SYNTHETIC: 4 = the generic sweep, 7 = wf_syn (the default
                           at skew 1), 8 = plane-split wf_syn (dsize 2..8, lane_cols = warps = skew = 1:
                           one warp per float item on the same 32 columns).  Other combinations
                           -> WF_EUNSUPPORTED */
  int32_t halo;         /* NEXT-4 comparison variant (PAPER.md P:238-255, P:289-296,
                           Table 3): columns each slab g > 0 recomputes redundantly west of its own
                           (an overlap of whole bands: a multiple of the band width); slab g then takes
                           its west input from slab g-1's column c0 - halo - 1 instead of c0 - 1, and the
                           overlap's cells go to a library scratch plane (outputs are unchanged).  SEQCMP
                           global alignment with the generation-8 sweep, ngpus > 1 only; 0 = none.
                           WF_EINVAL if not a positive multiple of the band width or if a slab has no
                           band to spare; WF_EUNSUPPORTED for other functions / generations */
  int32_t reserved[3];  /* must be zero */
} wf_params;

/* Distribution: which slab this context computes.
 *   single process, one slab:       dist = NULL  (slab 0 of 1, current device)
 *   single process, several slabs:  one context per slab, same or different devices; link them
 *                                   with wf_link_local(ctx[g], ctx[g+1])
 *   one process per GPU:            rank/world set; exchange wf_ipc_handle() bytes through the
 *                                   process group, then wf_connect(ctx, handle of rank+1). */
typedef struct {
  int32_t rank;         /* slab index g, 0 <= g < world */
  int32_t world;        /* number of slabs G (must equal params.ngpus) */
  int32_t device;       /* CUDA device ordinal for this slab; -1 = current device */
  int32_t device_share; /* contexts that run CONCURRENTLY on this device (virtual slabs share one
                           GPU); the persistent grid takes 1/device_share of the resident CTAs.
                           0 or 1 = exclusive. */
} wf_dist;

/* Per-slab layout (wf_query). */
typedef struct {
  int32_t nplanes;                 /* output planes */
  int32_t plane_bytes[WF_MAX_PLANES];  /* bytes per element of each plane (4) */
  int32_t plane_is_float[WF_MAX_PLANES];
  int32_t nbound;                  /* boundary planes expected in wf_io.top/left */
  int32_t col_begin, col_end;      /* this slab's interior columns [col_begin, col_end), 0-based */
  int64_t min_pitch;               /* minimum out_pitch in elements (slab columns rounded up to 4) */
  int64_t bytes_out;               /* bytes of all output planes at min_pitch */
  int32_t lane_cols, warps, skew;  /* effective tunables after defaults */
  int32_t band_cols;               /* columns per CTA band = warps * 32 * lane_cols (NASH: warps) */
  int32_t nbands;                  /* bands in this slab */
  int32_t strip;                   /* rows per hand-off block of the kernel that runs (generation 8);
                                      0 = fixed by the generation */
  int32_t reserved[4];
} wf_layout;

/* Device buffers for one wf_run.  All pointers are DEVICE pointers on the slab's device,
 * caller-owned, and must stay valid until the run completes on the stream.
 *   row_in : rows elements   (SEQCMP: uint8 codes x_i; SYNTHETIC: fp32 u_i; NASH: uint32 r_i)
 *   col_in : cols elements of the WHOLE grid (SEQCMP: uint8 y_j; SYNTHETIC: fp32 v_j; NASH: uint32 c_j)
 *   top[p] : boundary row 0 of plane p, cols+1 elements (index j = 0..cols; [0] is the corner)
 *   left[p]: boundary column 0 of plane p, rows+1 elements (index i; [0] ignored)
 *            p < nbound: SYNTHETIC nbound = dsize (the fp32 items; ints are fixed -1 / 0),
 *            NASH nbound = 4, SEQCMP nbound = 0 (boundary implied by gap).
 *   out[p] : plane p of this slab, rows x (col_end - col_begin) row-major, pitch out_pitch
 *            elements (multiple of 4, >= min_pitch), 16-byte aligned.  Padding columns are
 *            not written. */
typedef struct {
  const void* row_in;
  const void* col_in;
  const void* top[WF_MAX_PLANES];
  const void* left[WF_MAX_PLANES];
  void* out[WF_MAX_PLANES];
  int64_t out_pitch;
} wf_io;

/* Layout of rank's slab for params p (no device work).  WF_EINVAL on bad params. */
wf_status wf_query(const wf_params* p, int32_t rank, wf_layout* out);

/* Create a context: validates p, selects the device, allocates the library-owned scratch
 * (edge rings, error word) and sizes the persistent grid.  dist = NULL means 1 slab on the
 * current device.  On failure *out = NULL and wf_last_error(NULL) holds the message. */
wf_status wf_create(const wf_params* p, const wf_dist* dist, struct wf_ctx** out);

/* Enqueue one sweep of this slab on cuda_stream (a cudaStream_t; NULL = legacy default
 * stream).  Asynchronous, no host synchronisation; re-runnable with new inputs.  Reports a
 * device error left by the previous run (WF_ETIMEOUT) if it has already been observed. */
wf_status wf_run(struct wf_ctx* c, const wf_io* io, void* cuda_stream);

/* Block until this context's last run finished; returns WF_ETIMEOUT if a watchdog fired,
 * WF_ECUDA on a device fault. */
wf_status wf_sync(struct wf_ctx* c);

/* Free library-owned memory.  NULL-safe.  Never frees caller buffers. */
wf_status wf_destroy(struct wf_ctx* c);

/* Per-context message of the last failure; c == NULL -> last wf_create/wf_query failure of
 * this thread.  Never NULL. */
const char* wf_last_error(const struct wf_ctx* c);

/* Single-process multi-slab: make `next` (slab g+1) the consumer of `prev` (slab g).
 * Enables peer access when the devices differ (WF_ECOMM if impossible).  WF_EINVAL unless the two
 * contexts describe the same problem and tuning with prev's last column adjacent to next's first;
 * WF_ESTATE if either context has already run (linked slabs pair their runs by epoch: link first,
 * then issue the same sequence of wf_run calls on every slab). */
wf_status wf_link_local(struct wf_ctx* prev, struct wf_ctx* next);

/* One process per GPU: export this context's exchange buffer (control word + inbound edge
 * ring, one cudaMalloc) as a CUDA IPC handle (WF_IPC_HANDLE_BYTES bytes written to `handle`). */
wf_status wf_ipc_handle(struct wf_ctx* c, void* handle);

/* One process per GPU: open the neighbours' exchange buffers from their handle bytes; must be
 * called before the context's first wf_run (WF_ESTATE otherwise), and every rank then issues
 * the same sequence of wf_run calls (a rank that runs more often than its neighbour waits for
 * words that never come and reports WF_ETIMEOUT).
 * prev_handle: rank-1's handle (NULL on rank 0) -- this slab acknowledges each drained run
 * into it.  next_handle: rank+1's handle (NULL on the last rank) -- this slab's east edge is
 * stored into its ring over NVLink.  WF_EINVAL if a required handle is missing, WF_ECOMM if
 * a handle cannot be opened. */
wf_status wf_connect(struct wf_ctx* c, const void* prev_handle, const void* next_handle);

/* transport = WF_TRANSPORT_NCCL ("data elements have to be first transferred to the
 * host ... then to respective destination GPUs"; SURVEY.md §8(a) a8 "Fallback: NCCL send/recv"):
 * the slab-edge message of a staged context.
 *   wf_edge_bytes:  size of one message (the byte image of a band-0 edge ring; identical on all
 *                   ranks of one problem and tuning).
 *   wf_edge_export: rank < world-1: enqueue on `cuda_stream` a copy of the east edge written by
 *                   this slab's last wf_run into `dst` (device or pinned host memory, bytes from
 *                   wf_edge_bytes, caller-owned); call after wf_run on the same stream.
 *   wf_edge_import: rank > 0: enqueue a copy of the predecessor's exported message `src` into this
 *                   slab's inbound ring; call before wf_run on the same stream.
 * Every rank issues the same sequence of wf_run calls.  WF_ESTATE for a context that is not
 * staged (transport P2P, or a single slab) or for the wrong end of the chain; WF_EINVAL for
 * NULL pointers; WF_ECUDA if the copy cannot be enqueued. */
wf_status wf_edge_bytes(const struct wf_ctx* c, size_t* bytes);
wf_status wf_edge_export(struct wf_ctx* c, void* dst, void* cuda_stream);
wf_status wf_edge_import(struct wf_ctx* c, const void* src, void* cuda_stream);

/* SEQCMP local = 1 (Smith-Waterman): the best local
 * alignment score of this slab's columns and its cell, the first in row-major order holding
 * it -- 1-based row, 1-based GLOBAL column (a multi-slab caller takes the max over slabs,
 * ties to the smallest (row, col)).  Blocks until the last run completed.  WF_ESTATE if the
 * context is not local SEQCMP or has not run. */
wf_status wf_local_best(struct wf_ctx* c, int32_t* score, int32_t* row, int32_t* col);

/* Device time of the last completed run in milliseconds (CUDA events bracketing the
 * launch on the run's stream); WF_ESTATE if no run has completed. */
wf_status wf_last_run_ms(struct wf_ctx* c, float* ms);

/* Diagnostics: when the process runs with WF_TRACE=1, each wf_run records per band a
 * timeline of %globaltimer stamps (ns) taken by the band's first lane every rows/32 rows
 * (slots 0..31), at its last row (slot 32), and the feeder's poll / empty-poll counts
 * (slots 40, 41).  Copies min(bytes, nbands*slots*8) bytes of the last run to host;
 * *slots_per_band receives the slot count.  WF_ESTATE if tracing was not enabled. */
wf_status wf_debug_trace(struct wf_ctx* c, void* host, size_t bytes, int32_t* slots_per_band);

/* Library build information: ABI version, compiled arch, kernel variant count. */
int32_t wf_abi_version(void);
const char* wf_build_info(void);

#ifdef __cplusplus
}
#endif
#endif /* WF_H */
