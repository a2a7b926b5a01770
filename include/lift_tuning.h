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

#ifdef __cplusplus
}
#endif
#endif /* LIFT_TUNING_H */
