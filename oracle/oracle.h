/*
 * oracle.h — the CPU oracle for the SkelCL hot path (Steuwer & Gorlatch, PaCT 2013).
 *
 * TEST INFRASTRUCTURE ONLY.  Only tests/, __graft_entry__.smoke() and the
 * cpu_baseline / --impl reference legs of bench.py may load liboracle.so.  The
 * product path (libskl.so and its Python binding) never includes, links or calls
 * anything in oracle/, and nothing here includes anything from the product
 * (paper_conf_pact_steuwerg13_b200/csrc).
 *
 * Plain, slow, obviously-correct, single-threaded.  Every function cites the
 * PAPER.md line range (P:Lx-y) or the DESIGN.md reading (A<n>, from SURVEY.md
 * §8(c3)) it follows.  Built with -O2 -ffp-contract=off -fno-fast-math so that a
 * float expression is evaluated exactly as written (no FMA contraction): this is
 * the CPU twin of NVRTC's -fmad=false.
 *
 * fp32 Reduce/Scan with + accumulate in double; integer ops wrap
 * modulo 2^32 (A28, done in uint32_t).
 *
 * Parity status per function is listed in DESIGN.md §"Oracle pins".  The LM OSEM
 * functions (proposed workload A29, not in PAPER.md) are pinned only by
 * invariants and brute force: "parity unpinned by the paper".
 */
#ifndef SKL_ORACLE_H
#define SKL_ORACLE_H
#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

/* ---- Map -------------------------------------------------- */
enum oracle_map_fn {
  OM_NEG_F32 = 0,     /* "float func(float x){ return -x;}"            */
  OM_SQP1_F32 = 1,    /* x*x + 1.0f  (two roundings: pins -fmad=false)           */
  OM_INV_U8 = 2,      /* 255 - x                                               */
  OM_AFFINE_I32 = 3,  /* 3*x + 7 mod 2^32 (A28)                                */
};
int oracle_map(int fn, const void* in, void* out, size_t n);

/* Mandelbrot as a Map over complex numbers (A22, A23).
 * c is interleaved (re, im) float pairs; out[i] = escape iteration count.
 * Returns sum of iteration counts (the work unit of the bench).               */
uint64_t oracle_mandelbrot(const float* c, uint32_t* out, size_t npix, uint32_t max_iter);
/* row sums of the iteration counts of a rows x cols result (for imbalance)     */
void oracle_row_sums(const uint32_t* counts, size_t rows, size_t cols, uint64_t* sums);

/* ---- Zip -------------------------------------------------- */
enum oracle_zip_fn {
  OZ_ADD_F32 = 0,   /* "float func(float x,float y){return x+y;}" P:L261       */
  OZ_MULT_F32 = 1,  /* "float mult(float x,float y){return x*y;}" P:L290-291   */
  OZ_SUB_I32 = 2,   /* x - y mod 2^32                                          */
};
int oracle_zip(int fn, const void* l, const void* r, void* out, size_t n);

/* ---- Reduce and Scan ------------------------- */
enum oracle_op {
  OP_ADD_F32 = 0,    /* x+y on float, accumulated in double; result is double   */
  OP_ADD_I32 = 1,    /* x+y mod 2^32                                            */
  OP_MAX_F32 = 2,    /* fmaxf-free: (x > y ? x : y)                             */
  OP_LEFT_F32 = 3,   /* x (left projection; associative, not commutative)      */
  OP_RIGHT_F32 = 4,  /* y (right projection)                                    */
  OP_AFFINE_U32 = 5, /* (a1,b1)+(a2,b2) = (a1*a2, b1*a2+b2) mod 2^32; elements are
                        uint32 pairs: composition "first map 1, then map 2"     */
};
/* Left fold acc = v[0]; acc = acc (+) v[i].  n == 0 -> returns -1 (A11).
 * out holds one element of the result type (double for OP_ADD_F32).           */
int oracle_reduce(int op, const void* in, size_t n, void* out);
/* Inclusive scan out[0] = v[0]; out[i] = out[i-1] (+) v[i]  (A9).
 * out has the result type (double for OP_ADD_F32).                             */
int oracle_scan(int op, const void* in, size_t n, void* out);
/* Element-wise fold of G replicas in GPU order 0..G-1 (copy(+)->block, A25).
 * replicas is [G][n] of the op's element type, out is [n] of the result type. */
int oracle_combine(int op, const void* replicas, int G, size_t n, void* out);

/* ---- MapOverlap ------------------------------------------- */
enum oracle_stencil {
  OS_IDENT = 0,    /* get(0,0)                                                  */
  OS_SHIFT_X = 1,  /* get(+1,0): dx is the column offset (A15)                  */
  OS_SHIFT_Y = 2,  /* get(0,+1): dy is the row offset                           */
  OS_BOX3 = 3,     /* Listing 1.2 intended: sum over dx,dy in {-1,0,1} (A16), f32 */
  OS_SOBEL = 4,    /* Listing 1.5 / 1.4 with v = transpose of h (A17, A18), u8  */
  OS_GAUSS5 = 5,   /* 5x5 Gaussian sigma=1, proposed W1, f32                   */
};
enum oracle_boundary { OB_NEUTRAL = 0, OB_NEAREST = 1 };
/* type: 0 = u8, 1 = f32.  neutral points to one element of that type.         */
int oracle_mapoverlap2d(int stencil, int type, const void* in, void* out,
                        size_t rows, size_t cols, int d, int boundary, const void* neutral);
/* 1-D MapOverlap on a Vector: OS_IDENT, OS_SHIFT_X (get(+1)),
 * OS_BOX3 (sum of get(-1..1)), f32 only.                                       */
int oracle_mapoverlap1d(int stencil, const float* in, float* out, size_t n, int d,
                        int boundary, float neutral);
/* The 25 Gaussian weights the oracle uses, row-major [dy+2][dx+2]. */
void oracle_gauss5_weights(float* w25);

/* ---- Allpairs ----------------------------------------------- */
/* C[i][j] = A_i (+) B_j for rows A_i of the n x d matrix A and B_j of the m x d
 * matrix B.  The row function is a zip followed by a
 * left fold (reading A36): acc = z(a_0, b_0); acc = acc (+) z(a_k, b_k), k = 1..d-1
 *   AP_MANHATTAN  z = |a - b|, (+) = +   (the pairwise Manhattan distance)
 *   AP_DOT        z = a * b,   (+) = +   (dotProduct, Eq. (1))
 * in fp32 with every operation rounded (-ffp-contract=off); AP_DOT_F64 is the
 * same dot product accumulated in double (for the Eq. (2) pin A x B = allpairs(
 * dotProduct)(A, B^T)).  C is float (double for AP_DOT_F64).                   */
enum oracle_allpairs_fn { AP_MANHATTAN = 0, AP_DOT = 1, AP_DOT_F64 = 2 };
int oracle_allpairs(int fn, const float* A, const float* B, void* C, size_t n, size_t m, size_t d);

/* ---- Distributions (A1-A6, A25) ----------------------------- */
/* block: chunk = ceil(n/G); part g = [g*chunk, min((g+1)*chunk, n)) (A1)      */
void oracle_block_range(size_t n, int G, int g, size_t* lo, size_t* hi);
/* overlap(d): block range widened by d on each side, clipped to [0,n) (A3)    */
void oracle_overlap_range(size_t n, int G, int g, size_t d, size_t* lo, size_t* hi);

/* ---- LM OSEM (proposed workload W3, A29; not in PAPER.md) --------------- */
/* Siddon (1985) ray-voxel intersection of segment p0->p1 with the grid [0,N)^3
 * of unit voxels: all plane-crossing parameters alpha are merged and sorted; each
 * consecutive pair with positive length gives voxel at the midpoint.  Writes at
 * most cap entries; returns the number of segments.                            */
size_t oracle_siddon(const float* p0, const float* p1, int N, int64_t* vox, double* len, size_t cap);
/* One LM OSEM subset: for each event (x0,y0,z0,x1,y1,z1 floats),
 * fp = sum len*f[v]; if fp > 0: c[v] += len/fp.  Then fnew = f * c (sensitivity
 * 1).  c and fnew are double[N^3].  Returns #events with fp > 0; *visits = sum of
 * path lengths (voxel visits).                                                 */
uint64_t oracle_lmosem(const float* events, size_t nev, int N, const float* f,
                       double* c, double* fnew, uint64_t* visits);

#ifdef __cplusplus
}
#endif
#endif
