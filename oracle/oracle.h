/*
 * oracle.h — fp64 CPU oracle for the Lift zip->map->reduce hot path.
 *
 * TEST INFRASTRUCTURE ONLY.  Only tests/, __graft_entry__.smoke() and
 * bench.py's cpu_baseline / --impl reference leg may load this library.  It
 * shares no code, header, table or helper with the CUDA path
 * (paper_conf_cgo_steuwerrd17_b200/csrc, include/lift.h) and must never be
 * reached from the product path.
 *
 * Citations are PAPER.md line numbers (L<n>) of Steuwer, Remmelg, Dubach,
 * "Lift: A Functional Data-Parallel IR for High-Performance GPU Code
 * Generation", CGO 2017.
 *
 * Every reduction here is the plain sequential left fold of reduceSeq
 * (L320, Sec. 3.2: reduceSeq(z,f,x1..xn) = f(..f(f(z,x1),x2)..,xn)) with
 * z = 0, in fp64.  The product of two fp32 values is exact in fp64
 * (24+24 < 53 significand bits), so the only rounding is in the fp64 sum.
 * Each function also returns the tolerance magnitude "mag" (the sum of
 * |terms|) used by the acceptance test |y - y_ref| <= 1e-5*mag + 1e-6.
 *
 * Built with gcc -O2 -ffp-contract=off, never -ffast-math, so the compiler
 * neither contracts nor reassociates.  `threads` parallelises ONLY over
 * independent outputs (rows / column ranges); each output keeps its in-order
 * fold, so results are identical for every thread count.
 */
#ifndef LIFT_ORACLE_H
#define LIFT_ORACLE_H
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

/* dot(x, y) = reduce(+, 0, map(x, zip(x, y)))   — L285, Sec. 3.1 */
double oracle_dot(int64_t n, const float *x, const float *y, double *mag);

/* dot over all host cores (SURVEY.md 8(d) oracle timing variant (ii); reading
   R23): x*y cut into `chunks` fixed contiguous chunks (chunk k = elements
   [k*n/chunks, (k+1)*n/chunks)), each an in-order fp64 left fold, the chunk
   sums then folded in chunk order.  The grouping depends only on (n, chunks),
   never on `threads`, so every thread count gives the same bits; it differs
   from oracle_dot only in fp64 association (<= n * 2^-53 * mag). */
double oracle_dot_chunked(int64_t n, const float *x, const float *y, double *mag,
                          int chunks, int threads);

/* GEMV y = A x, A m x n row-major (lda = n)    — Table 1 L1030 (CLBlast GEMV);
   row i = join/split view of A (L329-334); reading A10 (row-major). */
void oracle_gemv(int64_t m, int64_t n, const float *A, const float *x,
                 double *y, double *mag, int threads);

/* GESUMMV y = alpha A x + beta B x            — Table 1; reading A9
   (PolyBench form: two sums, then combine).  alpha/beta are the fp32 values
   the C-ABI receives, widened exactly (reading A22). */
void oracle_gesummv(int64_t m, int64_t n, float alpha, const float *A,
                    float beta, const float *B, const float *x,
                    double *y, double *mag, int threads);

/* ATAX y = A^T (A x)                          — Table 1; reading A9.
   t = A x kept in fp64; y_j = sum_i A_ij t_i (transpose view L339-340,
   L848-850).  mag_j = sum_i |A_ij| * (sum_k |A_ik x_k|)  (reading A12). */
void oracle_atax(int64_t m, int64_t n, const float *A, const float *x,
                 double *y, double *mag, int threads);

/* partialDot, Listing 1 (L391-401): z[k] = sum_{i=chunk*k}^{chunk*k+chunk-1}
   x_i y_i for k < n/chunk (fp64 left fold).  Listing 1 uses chunk = 128
   (split128, L400); Fig. 7 drops a ragged tail (wg_id < N/128, L954). */
void oracle_partial_dot(int64_t n, int64_t chunk, const float *x,
                        const float *y, double *z, double *mag);

/* Listing 1 executed literally in fp32, in the paper's order:
   per work group k (mapWrg0 over split128, L392/L400), local thread l < 64
   (mapLcl0 over split2, L398-399) folds its pair with multAndSumUp
   (a + x*y, L767) from 0; then iterate6 (L394-397) halves 64 -> 1 with
   out[l] = reduceSeq(add, 0, [in[2l], in[2l+1]]).
   use_fma = 1: multAndSumUp = fmaf(x, y, a)   (one rounding)
   use_fma = 0: multAndSumUp = a + (float)(x*y) (two roundings)  — reading A2.
   Writes z[k], k < n/128. */
void oracle_partial_dot_listing1_f32(int64_t n, const float *x, const float *y,
                                     float *z, int use_fma);

/* The whole dot in the paper's structure (reading R26): Listing 1 over
   ceil(n/128) zero-padded chunks, then the same work-group program with add
   (the omitted second kernel, L422-426) applied repeatedly — iterate,
   L312-318 — until one value remains.  fp32, paper order. */
float oracle_dot_listing1_f32(int64_t n, const float *x, const float *y, int use_fma);

/* BLAS SGEMV (CLBlast contract, Table 1; NEXT-4):
   y = alpha*op(A) x + beta*y_in; layout 0 row-major A[i*lda+j], 1 column-major
   A[i+j*lda]; op = A (trans 0) or A^T (trans 1); beta == 0 does not read y_in. */
void oracle_sgemv(int layout, int trans, int64_t m, int64_t n, float alpha, const float *A, int64_t lda,
                  const float *x, float beta, const float *y_in, double *y, double *mag);

int oracle_version(void);

#ifdef __cplusplus
}
#endif
#endif
