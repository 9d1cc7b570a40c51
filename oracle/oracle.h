/*
 * oracle.h -- plain sequential CPU oracle for the wavefront sweep.
 *
 * TEST INFRASTRUCTURE ONLY.  Nothing on the product path (include/, the
 * paper_conf_ppopp_mohantyc14_b200 package, its CUDA library) may include,
 * link or call this.  Only tests/, __graft_entry__.smoke() and bench.py's
 * cpu_baseline leg / --impl reference arm use it.  It shares no code, header,
 * table or constant with the CUDA path.
 *
 * What it computes (Sec. 1, Fig. 1): "the values of the
 * relation are computed into a multidimensional array.  Computation starts at
 * position (0,0) and propagates to neighboring elements in a series of diagonal
 * bands".  The oracle evaluates the same relation in plain row-major order
 * (rows i = 1..m, columns j = 1..n), which is one topological order of the
 * dependency DAG a[i][j] = f(a[i-1][j], a[i][j-1], a[i-1][j-1]) (BASELINE.json
 * north_star).  Row 0 and column 0 are the boundary (reading R2).
 *
 * Output planes are row-major m x n (interior only), pitch n elements.
 * Every function returns 0 on success, -1 on a bad argument.
 */
#ifndef WF_ORACLE_H
#define WF_ORACLE_H
#include <stdint.h>
#ifdef __cplusplus
extern "C" {
#endif

/* Sequence comparison ("Biological Sequence Comparison [2]",
 * P:732 "Smith-Waterman"; BASELINE.json "Needleman-Wunsch integer scores").
 * x[0..m-1], y[0..n-1]: residue codes (any uint8; equality decides match).
 * local = 0: Needleman-Wunsch global alignment, linear gap g:
 *     H[i][0] = i*g, H[0][j] = j*g,
 *     H[i][j] = max(H[i-1][j-1] + s(x_i,y_j), H[i-1][j] + g, H[i][j-1] + g)
 * local = 1: Smith-Waterman local alignment: boundary 0 and max(..., 0).
 * H: m*n int32 output (rows 1..m_compute filled).  m_compute <= m limits the
 * work to a row prefix (0 = all rows). */
int oracle_seqcmp(int m, int n, int m_compute, const uint8_t* x, const uint8_t* y,
                  int32_t match, int32_t mismatch, int32_t gap, int local, int32_t* H);

/* Synthetic application (Sec. 3.1/3.1.1): each element is
 * two ints plus dsize floats; tsize is the per-element iteration count
 * (readings R4-R6).
 *   i0 = max(max(N.i0, NW.i0), W.i0) + 1
 *   i1 = ((N.i1 - NW.i1) + 1) + W.i1
 *   c  = (u_i * v_j) * 2^-12
 *   x_d = ((N.f[d] + NW.f[d]) + W.f[d]) * THIRD          THIRD = fp32 0x3EAAAAAB
 *   repeat tsize: x_d = fmaf(x_d, A, c)                    A = fp32 0x3F7FF000
 * Boundary: i0 = -1, i1 = 0 on row 0 and column 0; floats from top/left.
 * top: dsize arrays of n+1 floats (row 0, columns 0..n), packed as top[d*(n+1)+j].
 * left: dsize arrays of m+1 floats (column 0, rows 0..m), left[d*(m+1)+i];
 *       left[d*(m+1)+0] is ignored (the corner comes from top).
 * out_i0, out_i1: m*n int32; out_f: dsize planes of m*n floats, plane d at out_f + d*m*n. */
int oracle_synthetic(int m, int n, int m_compute, int tsize, int dsize,
                     const float* u, const float* v, const float* top, const float* left,
                     int32_t* out_i0, int32_t* out_i1, float* out_f);

/* Nash-equilibrium stand-in (reading R8).
 * Element = 4 int32 (p0..p3).  nstrat = n strategies per player (the nested
 * loop's granularity).  r[0..m-1], c[0..n-1] uint32 inputs.
 * top: 4 arrays of n+1 int32 (top[p*(n+1)+j]); left: 4 arrays of m+1 int32.
 * out: 4 planes of m*n int32, plane p at out + p*m*n. */
int oracle_nash(int m, int n, int m_compute, int nstrat, const uint32_t* r, const uint32_t* c,
                const int32_t* top, const int32_t* left, int32_t* out);

/* Test hooks for the Nash cell. */
uint32_t oracle_lowbias32(uint32_t x);
/* Pure-strategy Nash equilibria of the bimatrix game (A, B), both n x n row-major
 * (row player picks a, column player picks b).  out[0] = number of pure NE,
 * out[1] = smallest row-major index a*n+b of a pure NE (-1 if none),
 * out[2] = A at that index (-1), out[3] = B at that index (-1). */
int oracle_nash_solve(int nstrat, const int32_t* A, const int32_t* B, int32_t out[4]);
/* One Nash cell from its neighbours (exposes the key chain for tests). */
int oracle_nash_cell(int nstrat, const int32_t N[4], const int32_t NW[4], const int32_t W[4],
                     uint32_t r, uint32_t c, int32_t out[4]);

#ifdef __cplusplus
}
#endif
#endif
