/*
 * lift.h — C ABI of the B200-native Lift hot path:
 *          the fused zip -> map(x) -> reduce(+) kernel with no intermediate
 *          arrays, instantiated for dot, GEMV, GESUMMV and ATAX.
 *
 * Citations are PAPER.md line numbers (L<n>) of Steuwer, Remmelg, Dubach,
 * "Lift: A Functional Data-Parallel IR for High-Performance GPU Code
 * Generation", CGO 2017 (the file /root/reference/PAPER.md of the build).
 *
 * Conventions shared by every entry point
 * ---------------------------------------
 *  - Data: fp32 ("All experiments are performed using single precision
 *    floats", L1003).  Matrices are dense, row-major, contiguous, lda = n
 *    (reading R10).  Sizes are int64 (2^31-element configs; Fig. 7
 *    uses `int N`, L950 — widened, reading R7).
 *  - Pointers: every array pointer is a DEVICE pointer on the calling
 *    thread's current CUDA device, at least 4-byte aligned.  16-byte aligned
 *    bases with n % 4 == 0 take the 128-bit vector path (asVector4, L378-389);
 *    anything else takes the scalar path (same results contract).
 *  - Ownership: the caller owns every buffer.  The library never allocates,
 *    frees, synchronises, or changes the current device.
 *  - Streams: `stream` is a cudaStream_t (NULL = legacy default stream).
 *    Work is enqueued asynchronously; calls are CUDA-graph capturable.  The
 *    kernels (all but the fused collectives of lift_nvlink.h) are launched
 *    with programmatic stream serialisation
 *    (PDL): they may be scheduled while the previous kernel on the stream
 *    drains, but each waits for it (griddepcontrol.wait) before touching
 *    memory, so stream order is unchanged.  Before that wait a kernel may
 *    issue L2 prefetches (cp.async.bulk.prefetch.L2) of the first bytes of
 *    its read-only inputs; a prefetch delivers no data to the program and L2
 *    is the point of coherence, so an input the previous kernel is still
 *    writing is read only after the wait.  LIFT_PDL=0 in the environment
 *    turns it off.  Waits inside a kernel (grid barriers) are bounded by
 *    LIFT_SPIN_TIMEOUT_MS (default 20000) and trap when exceeded.
 *  - restrict: outputs must not overlap inputs or the workspace (Fig. 7
 *    declares `restrict` inputs, L948-950); overlap -> LIFT_ERR_ALIAS.
 *  - Errors: argument validation happens on the host BEFORE anything touches
 *    CUDA and returns a status with nothing enqueued.  LIFT_ERR_CUDA reports a
 *    launch/configuration error (text via lift_last_cuda_error()).  Faults
 *    during execution surface at the caller's next stream synchronisation.
 *  - Determinism: no floating-point atomics; for a fixed (shape, device) the
 *    output is bitwise reproducible.  GEMV/GESUMMV rows use one canonical
 *    summation order that depends only on n, so row-sharded results are
 *    bitwise equal to unsharded ones.
 *  - Accuracy contract (BASELINE.json north_star): elementwise
 *    |out - exact| <= 1e-5 * sum|terms| + 1e-6, fp32 accumulation in FMA.
 *  - Empty sizes: n == 0 -> dot writes 0, GEMV family writes y = 0 (m rows);
 *    m == 0 -> GEMV family is a no-op, ATAX writes y = 0 (n entries).
 */
#ifndef LIFT_H
#define LIFT_H

#include <stddef.h>
#include <stdint.h>

#if defined(__GNUC__)
#define LIFT_API __attribute__((visibility("default")))
#else
#define LIFT_API
#endif

#ifdef __cplusplus
extern "C" {
#endif

/* Same type as cudaStream_t, without requiring CUDA headers. */
typedef struct CUstream_st *lift_stream_t;

typedef enum lift_status {
    LIFT_OK = 0,
    LIFT_ERR_NULL_PTR = 1,   /* a pointer needed for a non-empty size is NULL          */
    LIFT_ERR_BAD_SIZE = 2,   /* negative size, m*n overflows int64, or size rule broken */
    LIFT_ERR_MISALIGNED = 3, /* a pointer is not 4-byte aligned                        */
    LIFT_ERR_ALIAS = 4,      /* an output range overlaps an input / workspace range    */
    LIFT_ERR_WORKSPACE = 5,  /* workspace NULL, too small, or not 16-byte aligned      */
    LIFT_ERR_CUDA = 6        /* CUDA launch / attribute error (lift_last_cuda_error()) */
} lift_status;

/* ---------------------------------------------------------------------- */
/* dot:  *result = sum_i x_i * y_i                                         */
/* ---------------------------------------------------------------------- */
/* dot(x, y) = reduce(+, 0, map(x, zip(x, y)))  — L285, Sec. 3.1; lowered as
 * Listing 1 (L391-401): per-thread reduceSeq(multAndSumUp, 0) over a chunk
 * (L398-399), an in-block tree (iterate6, L394-397) and a second stage over
 * the per-block results (L422-426) — here fused into ONE launch (the last
 * block to finish reduces the partials in a fixed order).
 *
 *   n          number of elements (>= 0)
 *   x, y       device fp32[n]
 *   result     device fp32[1], written (never read)
 *   workspace  device scratch of >= lift_dot_workspace_bytes(n) bytes,
 *              16-byte aligned.  Its first 16 bytes hold an arrival ticket
 *              that MUST be zero before the first call (e.g. cudaMemset once
 *              at allocation); every call leaves it zero again.  One
 *              workspace must not be used by concurrent calls.           */
LIFT_API size_t lift_dot_workspace_bytes(int64_t n);
LIFT_API int lift_dot(int64_t n, const float *x, const float *y, float *result,
             void *workspace, size_t workspace_bytes, lift_stream_t stream);

/* ---------------------------------------------------------------------- */
/* GEMV:  y = A x                                                          */
/* ---------------------------------------------------------------------- */
/* Table 1 GEMV (L1030; CLBlast, 4K^2 / 8K^2).  y_i is dot(A_i, x): rows are
 * distributed over blocks (mapWrg, L359-367) and x is staged once per block
 * in shared memory (toLocal, L368-377) by the bulk-copy (TMA) engine.
 * Reading R8: y = A x, y written and never read (BLAS alpha = 1, beta = 0).
 *
 *   m, n   rows, columns (>= 0)
 *   A      device fp32[m][n] row-major
 *   x      device fp32[n]
 *   y      device fp32[m], written                                       */
LIFT_API int lift_gemv(int64_t m, int64_t n, const float *A, const float *x, float *y,
              lift_stream_t stream);

/* ---------------------------------------------------------------------- */
/* GESUMMV:  y = alpha A x + beta B x                                      */
/* ---------------------------------------------------------------------- */
/* Table 1 GESUMMV (L1031).  Reading R9 (PolyBench): y = alpha*Ax + beta*Bx.
 * One kernel streams the zipped rows (A_i, B_i) (zip, L343-347) with two
 * accumulators; neither A x nor B x is materialised.  Epilogue per row:
 * y_i = alpha*sA + beta*sB, each product rounded, then one rounded add.
 *
 *   alpha, beta  fp32 scalars (by value)
 *   A, B         device fp32[m][n] row-major
 *   x            device fp32[n];  y device fp32[m], written              */
LIFT_API int lift_gesummv(int64_t m, int64_t n, float alpha, const float *A, float beta,
                 const float *B, const float *x, float *y, lift_stream_t stream);

/* ---------------------------------------------------------------------- */
/* ATAX:  y = A^T (A x)                                                    */
/* ---------------------------------------------------------------------- */
/* Table 1 ATAX (L1029).  Reading R9: t = A x (t in R^m, fp32), y = A^T t
 * (y in R^n).  The transpose is never materialised: A^T is read through the
 * transposed index l_id*N + wg_id (Fig. 6; matrixTranspose
 * L848-850).
 *
 * lift_atax picks the fastest algorithm for the shape:
 *   LIFT_ATAX_FUSED    one streaming pass over A: per row group, t_r = A_r x
 *                      by a block tree, then y_part += A_r^T t_r from the
 *                      same registers; then, in the same cooperative launch
 *                      after a grid barrier, a fixed-order reduce of the
 *                      per-block y_part (reads A once: 4*m*n bytes).
 *                      Needs 16-byte aligned A, x, y and n % 4 == 0; rows
 *                      of n <= 16384 are streamed by one block each (one
 *                      cooperative launch of one block per SM), wider rows
 *                      (n <= 262144, n a multiple of 4C whose slices are at
 *                      most 4096 float4) by a thread-block cluster of
 *                      C = 2..16 blocks over column slices (launched
 *                      cooperative with its cluster shape).  Other
 *                      shapes: LIFT_ERR_BAD_SIZE (auto uses TWOPASS).
 *                      The grid barrier's wait is bounded: if the blocks
 *                      could not all be resident it traps after the spin
 *                      limit (LIFT_SPIN_TIMEOUT_MS, default 20 s) and the
 *                      error surfaces at the next synchronisation.
 *   LIFT_ATAX_TWOPASS  the paper's structure (two GEMV-shaped kernels whose
 *                      times are summed, L1006-1007): GEMV t = A x, then a
 *                      column-blocked A^T t into per-row-split partials, then
 *                      a fixed-order reduce (reads A twice: 8*m*n bytes).
 *
 *   A          device fp32[m][n] row-major;  x device fp32[n]
 *   y          device fp32[n], written
 *   workspace  device scratch >= lift_atax_workspace_bytes(m, n), 16-byte
 *              aligned.  Its first 256 bytes hold grid-barrier counters that
 *              MUST be zero before the first call (cudaMemset once at
 *              allocation); every call leaves them zero.  Not shared by
 *              concurrent calls.                                          */
typedef enum lift_atax_algo {
    LIFT_ATAX_AUTO = 0,
    LIFT_ATAX_FUSED = 1,
    LIFT_ATAX_TWOPASS = 2
} lift_atax_algo;

LIFT_API size_t lift_atax_workspace_bytes(int64_t m, int64_t n);
LIFT_API int lift_atax(int64_t m, int64_t n, const float *A, const float *x, float *y,
              void *workspace, size_t workspace_bytes, lift_stream_t stream);
LIFT_API int lift_atax_algo_run(int algo, int64_t m, int64_t n, const float *A,
                       const float *x, float *y, void *workspace,
                       size_t workspace_bytes, lift_stream_t stream);

/* ---------------------------------------------------------------------- */
/* BLAS-complete GEMV (CLBlast SGEMV contract)                             */
/* ---------------------------------------------------------------------- */
/* Table 1's GEMV reference is CLBlast (L1030), whose SGEMV computes
 *     y = alpha * op(A) * x + beta * y,   op(A) = A (trans = 0) or A^T (trans = 1)
 * A is m x n with leading dimension lda:
 *     layout = 0 (row-major):    element (i, j) at A[i*lda + j], lda >= n
 *     layout = 1 (column-major): element (i, j) at A[i + j*lda], lda >= m
 * trans = 0: x in R^n, y in R^m;  trans = 1: x in R^m, y in R^n.
 * beta == 0: y is not read (BLAS convention: NaN/garbage in y is ignored).
 * A column-major matrix is the row-major transpose, so (layout 1, trans t)
 * runs the (layout 0, trans !t) kernels.  Non-transposed rows use the GEMV
 * kernel (canonical per-row order; alpha = 1, beta = 0 is bitwise lift_gemv);
 * transposed ones the column-blocked pass of two-pass ATAX + a fixed-order
 * column sum, with the epilogue y = alpha*s + beta*y (products rounded, then
 * one rounded add).
 *
 *   workspace  needed only for the transposed-row path:
 *              >= lift_sgemv_workspace_bytes(layout, trans, m, n) bytes,
 *              16-byte aligned (may be NULL when that is 0)             */
LIFT_API size_t lift_sgemv_workspace_bytes(int layout, int trans, int64_t m, int64_t n);
LIFT_API int lift_sgemv(int layout, int trans, int64_t m, int64_t n, float alpha,
                        const float *A, int64_t lda, const float *x, float beta, float *y,
                        void *workspace, size_t workspace_bytes, lift_stream_t stream);

/* ---------------------------------------------------------------------- */
/* Listing 1 in the paper's exact order (bitwise reproducible semantics)   */
/* ---------------------------------------------------------------------- */
/* partialDot (Listing 1; generated kernel Fig. 7):
 * work group k reduces the 128-element chunk k of zip(x, y): local thread l
 * (of 64) folds elements 2l, 2l+1 with multAndSumUp from 0, then iterate6
 * halves 64 -> 1 with out[l] = (0 + in[2l]) + in[2l+1].  Every fp32 operation
 * happens in exactly this order, so the result is a fixed bit pattern for
 * given inputs (pinned against oracle/ bit for bit).
 *
 *   n         elements (>= 0); z gets n/128 values (Fig. 7 forms only N/128
 *             work groups, L954; a ragged tail is ignored, as in the paper)
 *   x, y      device fp32[n], 4-byte aligned (16-byte alignment is faster)
 *   z         device fp32[n/128], written
 *   contract  1: multAndSumUp = fma(x, y, a) (one rounding);
 *             0: a + (x*y) with the product rounded first (reading R2)    */
LIFT_API int lift_partial_dot(int64_t n, const float *x, const float *y, float *z,
                              int contract, lift_stream_t stream);

/* The whole dot in the paper's structure (reading R26): Listing 1 over
 * ceil(n/128) zero-padded chunks, then the same work-group program with add
 * (the second kernel the paper omits, L422-426) applied again — iterate,
 * L312-318 — until one value remains: ceil(log128 n) launches.  Bitwise
 * equal to oracle_dot_listing1_f32.  n == 0 writes 0.
 *
 *   result     device fp32[1], written
 *   workspace  device scratch >= lift_dot_listing1_workspace_bytes(n),
 *              16-byte aligned, no initialisation needed                 */
LIFT_API size_t lift_dot_listing1_workspace_bytes(int64_t n);
LIFT_API int lift_dot_listing1(int64_t n, const float *x, const float *y, float *result,
                               void *workspace, size_t workspace_bytes, int contract,
                               lift_stream_t stream);

/* ---------------------------------------------------------------------- */
/* library info                                                            */
/* ---------------------------------------------------------------------- */
LIFT_API const char *lift_strerror(int status);      /* static string, never NULL   */
LIFT_API const char *lift_last_cuda_error(void);     /* thread-local, last CUDA error text */
LIFT_API int lift_version(void);                     /* (major << 16) | minor        */

#ifdef __cplusplus
}
#endif
#endif /* LIFT_H */
