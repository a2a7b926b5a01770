/*
 * lift_nvlink.h — the sharded ops with their collective fused into the
 * kernel: instead of a separate NCCL call, each rank's
 * kernel stores its results straight into every destination rank's
 * symmetric "exchange area" over NVLink (one-sided st.global on peer
 * pointers), publishes a per-(rank, epoch) flag with st.release.sys, and the
 * receiving side acquires all flags and combines the contributions in RANK
 * ORDER — so every receiving rank gets bitwise the same result, and the
 * transfer of a GEMV row overlaps the computation of the next ones.
 *
 * Exchange area: a device allocation of lift_exchange_bytes(...) bytes that
 * exists on EVERY rank with the same size (e.g. torch symmetric memory), ZERO
 * before its first use.  `peers` is a DEVICE array of `world` pointers: entry r
 * is rank r's exchange area as mapped in the calling process (entry `rank` is
 * the caller's own).  One exchange area serves one op at a time.
 *
 * Calls on one exchange area must be made in the same order on every rank
 * (every rank makes the matching call).  The call counter (epoch) lives in
 * the area on the device — the host passes none — so a sequence of these
 * calls can be captured in a CUDA graph and replayed.  Data is double
 * buffered by epoch parity; every call ends (on the device) only once every
 * rank has acknowledged reading the previous call's data, so the next call
 * never overwrites data a slower rank is still reading, in any mix of
 * all-reduce, all-gather and reduce-to-one-rank calls.
 * A rank that never makes the matching call makes its peers trap after the
 * spin limit (LIFT_SPIN_TIMEOUT_MS, default 20 s; the launch fails with a
 * CUDA error at the next synchronisation) instead of hanging the GPU.
 *
 * Validation follows lift.h (status codes, nothing enqueued on error); the
 * contents of `peers` live in device memory and are not checked.
 */
#ifndef LIFT_NVLINK_H
#define LIFT_NVLINK_H

#include "lift.h"

#ifdef __cplusplus
extern "C" {
#endif

typedef enum lift_exchange_kind {
    LIFT_EXCH_DOT = 0,      /* all-reduce of one fp32 per rank          */
    LIFT_EXCH_GATHER = 1,   /* all-gather of `len` = total rows of y    */
    LIFT_EXCH_REDUCE = 2    /* (all-)reduce of world partial rows of `len` = n floats */
} lift_exchange_kind;

LIFT_API size_t lift_exchange_bytes(int kind, int64_t len, int world);

/* dot over element slices: *result = sum over ranks of dot(x_r, y_r), summed
 * in rank order, identical on every rank.  workspace as in lift_dot.      */
LIFT_API int lift_dot_allreduce(int64_t n, const float *x, const float *y, float *result,
                                void *workspace, size_t workspace_bytes,
                                void *const *peers, int rank, int world,
                                lift_stream_t stream);

/* GEMV / GESUMMV over row blocks: rank `rank` holds rows [row0, row0+m) of
 * the m_total-row matrix; on return (stream order) y[0..m_total) holds the
 * full result on every rank, bitwise equal to the unsharded lift_gemv /
 * lift_gesummv.  workspace: >= 16 bytes, 16-byte aligned, zero before the
 * first call (an arrival ticket, re-armed by every call).                  */
LIFT_API int lift_gemv_allgather(int64_t m, int64_t n, const float *A, const float *x,
                                 int64_t row0, int64_t m_total, float *y,
                                 void *workspace, size_t workspace_bytes,
                                 void *const *peers, int rank, int world,
                                 lift_stream_t stream);
LIFT_API int lift_gesummv_allgather(int64_t m, int64_t n, float alpha, const float *A, float beta,
                                    const float *B, const float *x, int64_t row0, int64_t m_total,
                                    float *y, void *workspace, size_t workspace_bytes,
                                    void *const *peers, int rank, int world,
                                    lift_stream_t stream);

/* ATAX over row blocks: y = sum over ranks of A_r^T (A_r x) on rank `dst`
 * (dst = -1: on every rank), computed by the single-pass fused kernel (needs
 * n % 4 == 0, 16-byte aligned A, x, y, 256 <= n <= 16384); m may be 0.
 * On a non-destination rank y receives that rank's own partial.
 * workspace: as lift_atax.  blocks: 0 = one block per SM with a cooperative
 * launch; > 0 = that many blocks, plain launch (for running several ranks on
 * one GPU in tests: the caller guarantees co-residency).                  */
LIFT_API int lift_atax_reduce(int64_t m, int64_t n, const float *A, const float *x, float *y,
                              void *workspace, size_t workspace_bytes,
                              void *const *peers, int rank, int world, int dst,
                              int blocks, lift_stream_t stream);

#ifdef __cplusplus
}
#endif
#endif /* LIFT_NVLINK_H */
