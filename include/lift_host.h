/*
 * lift_host.h — the four ops end to end from HOST buffers: each call
 * enqueues, on `stream`, the host->device copies of its inputs, the same
 * kernels as lift.h, and the device->host copy of its result.  This is the
 * path the benchmark's "e2e" number measures (BASELINE.json metric, inputs
 * NOT resident in HBM), and the one a caller with host data uses.
 *
 * Conventions (in addition to lift.h):
 *  - *_host pointers are HOST memory.  Pinned (cudaHostAlloc / page-locked)
 *    memory makes every copy asynchronous; pageable memory is accepted but
 *    the copies then synchronise with the host (CUDA semantics).
 *  - *_dev pointers are caller-owned DEVICE buffers of the operand sizes that
 *    receive the copies (the library still never allocates).
 *  - The result is in *_host only after the stream is synchronised.
 *  - Validation is as in lift.h, plus: a device buffer may not overlap
 *    another one (LIFT_ERR_ALIAS).
 */
#ifndef LIFT_HOST_H
#define LIFT_HOST_H

#include "lift.h"

#ifdef __cplusplus
extern "C" {
#endif

/* *result_host = dot(x, y) (lift_dot) */
LIFT_API int lift_dot_host(int64_t n, const float *x_host, const float *y_host, float *result_host,
                           float *x_dev, float *y_dev, float *result_dev,
                           void *workspace, size_t workspace_bytes, lift_stream_t stream);

/* y_host = A x (lift_gemv) */
LIFT_API int lift_gemv_host(int64_t m, int64_t n, const float *A_host, const float *x_host, float *y_host,
                            float *A_dev, float *x_dev, float *y_dev, lift_stream_t stream);

/* y_host = alpha A x + beta B x (lift_gesummv) */
LIFT_API int lift_gesummv_host(int64_t m, int64_t n, float alpha, const float *A_host, float beta,
                               const float *B_host, const float *x_host, float *y_host,
                               float *A_dev, float *B_dev, float *x_dev, float *y_dev,
                               lift_stream_t stream);

/* y_host = A^T (A x) (lift_atax, automatic algorithm) */
LIFT_API int lift_atax_host(int64_t m, int64_t n, const float *A_host, const float *x_host, float *y_host,
                            float *A_dev, float *x_dev, float *y_dev,
                            void *workspace, size_t workspace_bytes, lift_stream_t stream);

#ifdef __cplusplus
}
#endif
#endif /* LIFT_HOST_H */
