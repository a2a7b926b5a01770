/*
 * lift_tuning.h — launch-configuration overrides for benchmarking and
 * tuning sweeps.  Same contract as the corresponding entry points in lift.h
 * (validation, ownership, streams, errors); results are bitwise identical to
 * the untuned calls for every accepted configuration (GEMV rows use one
 * canonical summation order, see lift.h), only the speed changes.
 *
 *   wpr     warps cooperating on one row: 1, 2, 4 or 8 (0 = automatic)
 *   rg      rows in flight per block:  wpr*rg*32 threads per block must be
 *           one of the compiled shapes (wpr,rg) in {(8,1),(8,2),(4,2),(4,4),
 *           (2,4),(2,8),(1,8)} (0 = automatic)
 *   blocks  grid size (0 = persistent grid sized from the SM count)
 *   xsmem   1 = stage x in shared memory with the bulk-copy engine,
 *           0 = read x through the L1 cache, -1 = automatic
 *   lb      vector loads per lane per batch, 4 or 8 (the kernel keeps two
 *           batches in flight); 0 = automatic
 * The scalar path (n % 4 != 0 or a base not 16-byte aligned) has one shape:
 * wpr = 1, rg = 8, lb = 4 (or 0 for each).
 *
 * lift_atax_fused_tuned: lift_atax with the single-pass fused kernel
 * (lift_atax_algo_run(LIFT_ATAX_FUSED, ...): same arguments, workspace and
 * validation):
 *   nst       stages in the shared-memory ring (one bulk copy of ~32 KiB of
 *             rows each up to 16384 columns, one row slice each for the
 *             wider, cluster kernel), 2..16 and within the shared-memory
 *             budget (0 = automatic).  Only the speed changes: results are
 *             bitwise those of lift_atax_algo_run(LIFT_ATAX_FUSED, ...) for
 *             every accepted nst, at every width.
 *   cyclic    1 = block b streams row stages b, b+G, b+2G, ... (G blocks),
 *             0 = block b streams one contiguous band of rows (-1 = automatic,
 *             which is 1).  This changes which rows each block's partial sums,
 *             so results are bitwise those of the untuned call only at 1 / -1.
 *             Rows wider than 16384 (the cluster kernel) are always assigned
 *             cyclically: 0 is refused there.
 *
 * An unsupported combination returns LIFT_ERR_CUDA with
 * lift_last_cuda_error() = "invalid argument".
 */
#ifndef LIFT_TUNING_H
#define LIFT_TUNING_H

#include "lift.h"

#ifdef __cplusplus
extern "C" {
#endif

LIFT_API int lift_gemv_tuned(int64_t m, int64_t n, const float *A, const float *x, float *y,
                    int wpr, int rg, int blocks, int xsmem, int lb, lift_stream_t stream);

LIFT_API int lift_gesummv_tuned(int64_t m, int64_t n, float alpha, const float *A, float beta,
                       const float *B, const float *x, float *y,
                       int wpr, int rg, int blocks, int xsmem, int lb, lift_stream_t stream);

LIFT_API int lift_atax_fused_tuned(int64_t m, int64_t n, const float *A, const float *x, float *y,
                                   void *workspace, size_t workspace_bytes, int nst, int cyclic,
                                   lift_stream_t stream);

/* lift_atax_fused_grid: the launch shape of lift_atax's single pass for an
 * m x n matrix on the current device, without launching anything: *blocks
 * thread blocks in clusters of *cluster (1 = no cluster: one block per SM,
 * rows up to 16384 wide, a cooperative launch; 2..16 = the wide-row kernel,
 * as many clusters as the device's cluster occupancy allows — the GPC layout
 * of the part decides it —, launched cooperative with its cluster shape).
 * LIFT_ERR_BAD_SIZE for shapes the single pass does not take (m < 1, n not a
 * supported width), LIFT_ERR_NULL_PTR for NULL outputs, LIFT_ERR_CUDA when
 * there is no device. */
LIFT_API int lift_atax_fused_grid(int64_t m, int64_t n, int *blocks, int *cluster);

#ifdef __cplusplus
}
#endif
#endif /* LIFT_TUNING_H */
