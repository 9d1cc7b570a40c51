/*
 * oracle.c -- plain, slow, obviously correct sequential CPU oracle.
 *
 * TEST INFRASTRUCTURE ONLY (see oracle.h).  Single thread, row-major loop,
 * built with -O2 -ffp-contract=off (no FMA contraction, no fast-math, default
 * MXCSR: no FTZ/DAZ) so each float operation below is exactly one IEEE-754
 * binary32 round-to-nearest operation (reading R11).
 *
 * Every function follows the definition it cites; there is no blocking,
 * fusion or reordering.  The boundary accessors make the neighbour reads
 * a[i-1][j], a[i][j-1], a[i-1][j-1] literal.
 */
#include "oracle.h"

#include <math.h>
#include <stddef.h>
#include <string.h>

/* ------------------------------------------------------------------------ */
/* Sequence comparison: Needleman-Wunsch (global) / Smith-Waterman (local).   */
/* PAPER.md P:432-435 (app), P:732 (named Smith-Waterman), BASELINE.json       */
/* configs ("Needleman-Wunsch integer scores"); readings R9, R10.    */
/* ------------------------------------------------------------------------ */

/* H(i,j) for 0 <= i <= m, 0 <= j <= n; interior from the output array. */
static int32_t seq_get(const int32_t* H, int n, int32_t gap, int local, int i, int j) {
  if (i == 0) return local ? 0 : (int32_t)j * gap;   /* H[0][j] = j*g (NW), 0 (SW) */
  if (j == 0) return local ? 0 : (int32_t)i * gap;   /* H[i][0] = i*g (NW), 0 (SW) */
  return H[(size_t)(i - 1) * n + (j - 1)];
}

static int32_t max2(int32_t a, int32_t b) { return a > b ? a : b; }

int oracle_seqcmp(int m, int n, int m_compute, const uint8_t* x, const uint8_t* y,
                  int32_t match, int32_t mismatch, int32_t gap, int local, int32_t* H) {
  if (m < 0 || n < 0 || !H || (m > 0 && !x) || (n > 0 && !y)) return -1;
  if (m_compute <= 0 || m_compute > m) m_compute = m;
  for (int i = 1; i <= m_compute; ++i) {
    for (int j = 1; j <= n; ++j) {
      int32_t N = seq_get(H, n, gap, local, i - 1, j);
      int32_t W = seq_get(H, n, gap, local, i, j - 1);
      int32_t NW = seq_get(H, n, gap, local, i - 1, j - 1);
      int32_t s = (x[i - 1] == y[j - 1]) ? match : mismatch;
      int32_t h = max2(max2(NW + s, N + gap), W + gap);
      if (local) h = max2(h, 0);
      H[(size_t)(i - 1) * n + (j - 1)] = h;
    }
  }
  return 0;
}

/* ------------------------------------------------------------------------ */
/* Synthetic application.  PAPER.md P:349-375 (Sec. 3.1.1): "tsize is measured */
/* in units of the execution time of a single iteration of the synthetic      */
/* kernel function"; "each element ... consists of two int variables and a    */
/* varying number of floats, controlled by dsize".  The body is not given in  */
/* the paper; readings R4-R6 fix it.                                */
/* ------------------------------------------------------------------------ */

static float f32_from_bits(uint32_t b) { float f; memcpy(&f, &b, 4); return f; }

typedef struct { int32_t i0, i1; } syn_ints;

static syn_ints syn_get_ints(const int32_t* I0, const int32_t* I1, int n, int i, int j) {
  syn_ints r;
  if (i == 0 || j == 0) { r.i0 = -1; r.i1 = 0; return r; }   /* boundary ints */
  r.i0 = I0[(size_t)(i - 1) * n + (j - 1)];
  r.i1 = I1[(size_t)(i - 1) * n + (j - 1)];
  return r;
}

static float syn_get_f(const float* F, const float* top, const float* left, int m, int n, int d,
                       int i, int j) {
  if (i == 0) return top[(size_t)d * (n + 1) + j];           /* row 0, incl. corner */
  if (j == 0) return left[(size_t)d * (m + 1) + i];          /* column 0, i >= 1 */
  return F[(size_t)d * m * n + (size_t)(i - 1) * n + (j - 1)];
}

int oracle_synthetic(int m, int n, int m_compute, int tsize, int dsize,
                     const float* u, const float* v, const float* top, const float* left,
                     int32_t* out_i0, int32_t* out_i1, float* out_f) {
  if (m < 0 || n < 0 || tsize < 0 || dsize < 0 || !out_i0 || !out_i1) return -1;
  if (dsize > 0 && (!top || !left || !out_f || !u || !v)) return -1;
  if (m_compute <= 0 || m_compute > m) m_compute = m;
  const float THIRD = f32_from_bits(0x3EAAAAABu);   /* fp32 nearest to 1/3 */
  const float A = f32_from_bits(0x3F7FF000u);       /* 1 - 2^-12 */
  const float SCALE = f32_from_bits(0x39800000u);   /* 2^-12 */
  for (int i = 1; i <= m_compute; ++i) {
    for (int j = 1; j <= n; ++j) {
      syn_ints N = syn_get_ints(out_i0, out_i1, n, i - 1, j);
      syn_ints W = syn_get_ints(out_i0, out_i1, n, i, j - 1);
      syn_ints NW = syn_get_ints(out_i0, out_i1, n, i - 1, j - 1);
      int32_t i0 = max2(max2(N.i0, NW.i0), W.i0) + 1;
      int32_t i1 = ((N.i1 - NW.i1) + 1) + W.i1;
      out_i0[(size_t)(i - 1) * n + (j - 1)] = i0;
      out_i1[(size_t)(i - 1) * n + (j - 1)] = i1;
      if (dsize > 0) {
        float uv = u[i - 1] * v[j - 1];                /* one RN multiply */
        float c = uv * SCALE;                           /* exact power-of-two scale */
        for (int d = 0; d < dsize; ++d) {
          float fN = syn_get_f(out_f, top, left, m, n, d, i - 1, j);
          float fW = syn_get_f(out_f, top, left, m, n, d, i, j - 1);
          float fNW = syn_get_f(out_f, top, left, m, n, d, i - 1, j - 1);
          float s1 = fN + fNW;
          float s2 = s1 + fW;
          float xd = s2 * THIRD;
          for (int t = 0; t < tsize; ++t) xd = fmaf(xd, A, c);
          out_f[(size_t)d * m * n + (size_t)(i - 1) * n + (j - 1)] = xd;
        }
      }
    }
  }
  return 0;
}

/* ------------------------------------------------------------------------ */
/* Nash-equilibrium application.  PAPER.md P:428-431: "A game-theoretic      */
/* problem ... very computationally demanding kernel.  The internal          */
/* granularity parameter controls the iteration count of a nested loop";     */
/* P:437-439 maps it to dsize = 4.  The kernel of ref. [15] is not given;    */
/* DESIGN.md reading R8 defines this integer stand-in.                        */
/* ------------------------------------------------------------------------ */

uint32_t oracle_lowbias32(uint32_t x) {
  x ^= x >> 16;
  x *= 0x7feb352du;
  x ^= x >> 15;
  x *= 0x846ca68bu;
  x ^= x >> 16;
  return x;
}

int oracle_nash_solve(int nstrat, const int32_t* A, const int32_t* B, int32_t out[4]) {
  if (nstrat < 1 || !A || !B || !out) return -1;
  int count = 0, first = -1;
  for (int a = 0; a < nstrat; ++a) {
    for (int b = 0; b < nstrat; ++b) {
      /* (a,b) is a pure Nash equilibrium iff neither player gains by deviating:
         A[a][b] >= A[a'][b] for all a', and B[a][b] >= B[a][b'] for all b'. */
      int best_for_row = 1, best_for_col = 1;
      for (int a2 = 0; a2 < nstrat; ++a2)
        if (A[a2 * nstrat + b] > A[a * nstrat + b]) best_for_row = 0;
      for (int b2 = 0; b2 < nstrat; ++b2)
        if (B[a * nstrat + b2] > B[a * nstrat + b]) best_for_col = 0;
      if (best_for_row && best_for_col) {
        if (first < 0) first = a * nstrat + b;
        ++count;
      }
    }
  }
  out[0] = count;
  out[1] = first;
  out[2] = first >= 0 ? A[first] : -1;
  out[3] = first >= 0 ? B[first] : -1;
  return 0;
}

#define NASH_SEED 0x9E3779B9u
#define NASH_MAXN 64

int oracle_nash_cell(int nstrat, const int32_t N[4], const int32_t NW[4], const int32_t W[4],
                     uint32_t r, uint32_t c, int32_t out[4]) {
  if (nstrat < 1 || nstrat > NASH_MAXN) return -1;
  /* key chain: N.p0..p3, NW.p0..p3, r_i, c_j, W.p0..p3 (W enters last) */
  uint32_t key = NASH_SEED;
  for (int p = 0; p < 4; ++p) key = oracle_lowbias32(key ^ (uint32_t)N[p]);
  for (int p = 0; p < 4; ++p) key = oracle_lowbias32(key ^ (uint32_t)NW[p]);
  key = oracle_lowbias32(key ^ r);
  key = oracle_lowbias32(key ^ c);
  for (int p = 0; p < 4; ++p) key = oracle_lowbias32(key ^ (uint32_t)W[p]);
  /* payoff matrices of the cell's game */
  static int32_t A[NASH_MAXN * NASH_MAXN], B[NASH_MAXN * NASH_MAXN];
  for (int a = 0; a < nstrat; ++a) {
    for (int b = 0; b < nstrat; ++b) {
      uint32_t idx = (uint32_t)(a * nstrat + b);
      A[idx] = (int32_t)(oracle_lowbias32(key ^ (2u * idx)) & 255u);
      B[idx] = (int32_t)(oracle_lowbias32(key ^ (2u * idx + 1u)) & 255u);
    }
  }
  return oracle_nash_solve(nstrat, A, B, out);
}

static void nash_get(const int32_t* out, const int32_t* top, const int32_t* left, int m, int n,
                     int i, int j, int32_t v[4]) {
  for (int p = 0; p < 4; ++p) {
    if (i == 0) v[p] = top[(size_t)p * (n + 1) + j];
    else if (j == 0) v[p] = left[(size_t)p * (m + 1) + i];
    else v[p] = out[(size_t)p * m * n + (size_t)(i - 1) * n + (j - 1)];
  }
}

int oracle_nash(int m, int n, int m_compute, int nstrat, const uint32_t* r, const uint32_t* c,
                const int32_t* top, const int32_t* left, int32_t* out) {
  if (m < 0 || n < 0 || nstrat < 1 || nstrat > NASH_MAXN || !out) return -1;
  if ((m > 0 && n > 0) && (!r || !c || !top || !left)) return -1;
  if (m_compute <= 0 || m_compute > m) m_compute = m;
  for (int i = 1; i <= m_compute; ++i) {
    for (int j = 1; j <= n; ++j) {
      int32_t N[4], W[4], NW[4], o[4];
      nash_get(out, top, left, m, n, i - 1, j, N);
      nash_get(out, top, left, m, n, i, j - 1, W);
      nash_get(out, top, left, m, n, i - 1, j - 1, NW);
      if (oracle_nash_cell(nstrat, N, NW, W, r[i - 1], c[j - 1], o) != 0) return -1;
      for (int p = 0; p < 4; ++p) out[(size_t)p * m * n + (size_t)(i - 1) * n + (j - 1)] = o[p];
    }
  }
  return 0;
}
