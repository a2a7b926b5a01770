// launch.h — internal launcher interface between capi.cu (validation,
// configuration) and the kernel translation units.  Not part of the C ABI.
#pragma once

#include <cuda_runtime.h>
#include <stddef.h>
#include <stdint.h>

#include "exchange.cuh"

namespace lift {

struct DeviceInfo {
    int device = -1;
    int sms = 0;              // cudaDevAttrMultiProcessorCount (148 on B200)
    int smem_optin = 0;       // max dynamic smem per block (opt-in)
    int smem_per_sm = 0;      // max smem per SM
    int max_threads_sm = 0;   // 2048
    int regs_per_sm = 0;      // 65536
};

// Cached per device; thread-safe after the first call per device.  The first
// call on a device also loads every kernel of the library (preload_*).
cudaError_t device_info(DeviceInfo *out);
cudaError_t preload_dot();
cudaError_t preload_gemv();
cudaError_t preload_atax();
cudaError_t preload_listing1();

// ---- dot -------------------------------------------------------------------
constexpr int kDotMaxBlocks = 4096;
constexpr size_t kDotTicketBytes = 16;
cudaError_t launch_dot(const DeviceInfo &d, int64_t n, const float *x, const float *y, float *result,
                       void *workspace, cudaStream_t s, Exch ex = Exch{});

// ---- GEMV / GESUMMV ----------------------------------------------------------
struct GemvConfig {
    int wpr = 0;     // warps per row   (1, 2, 4, 8); 0 = auto
    int rg = 0;      // row groups per block; 0 = auto
    int blocks = 0;  // grid size; 0 = auto (persistent)
    int xsmem = -1;  // 1 = stage x in smem by bulk copy, 0 = read x through L1, -1 = auto
    int lb = 0;      // vector loads per lane per batch (4 or 8; x2 in flight with the prefetch); 0 = auto
};
// Epilogue applied to the row sums (sA, sB):
//   kEpiStore   y_i = sA                                  (GEMV)
//   kEpiAxpby   y_i = alpha*sA + beta*y_i  (y not read when beta == 0; BLAS SGEMV)
//   kEpiSum2    y_i = alpha*sA + beta*sB                  (GESUMMV, nmat = 2)
// Each product is rounded, then one rounded add.
enum GemvEpi { kEpiStore = 0, kEpiAxpby = 1, kEpiSum2 = 2 };
struct GemvArgs {
    int nmat = 1;            // 1: A only; 2: A and B (zipped rows)
    int64_t m = 0, n = 0;    // rows, columns
    int64_t lda = 0;         // row stride of A and B in floats (>= n)
    const float *A = nullptr, *B = nullptr, *x = nullptr;
    float *y = nullptr;
    float alpha = 1.f, beta = 0.f;
    int epi = kEpiStore;
    // fused all-gather (NEXT-2): rows go to every rank's exchange area at row0 + i;
    // the last block waits for all ranks and copies the m_total gathered rows to y
    Exch ex;
    int64_t row0 = 0, m_total = 0;
    unsigned int *ticket = nullptr;  // zeroed once; re-armed by every launch
};
cudaError_t launch_gemv(const DeviceInfo &d, const GemvArgs &a, GemvConfig cfg, cudaStream_t s);

// ---- ATAX ----------------------------------------------------------------------
size_t atax_twopass_ws_bytes(int64_t m, int64_t n);
size_t atax_fused_ws_bytes(int64_t m, int64_t n);
bool atax_fused_supported(int64_t m, int64_t n, bool aligned16);
bool atax_fused_preferred(int64_t m, int64_t n, bool aligned16);
bool atax_fused_exchange_supported(int64_t m, int64_t n, bool aligned16);  // the NVLink-fused form (n <= 16384)
cudaError_t atax_fused_grid(const DeviceInfo &d, int64_t m, int64_t n, int *blocks, int *cluster);
cudaError_t launch_atax_twopass(const DeviceInfo &d, int64_t m, int64_t n, const float *A, const float *x,
                                float *y, void *ws, cudaStream_t s);
// y = alpha * A^T x + beta * y  (A m x n row-major with stride lda; x in R^m, y in R^n):
// column-blocked partials over row splits + fixed-order column sum with the epilogue
size_t gemv_t_ws_bytes(int64_t m, int64_t n);
cudaError_t launch_gemv_t(const DeviceInfo &d, int64_t m, int64_t n, int64_t lda, float alpha, const float *A,
                          const float *x, float beta, float *y, void *ws, cudaStream_t s);
// FusedTuning: nst = ring stages (0 = planned), cyc = 1 cyclic / 0 banded row
// assignment (-1 = planned; the wide-row kernel is always cyclic)
struct FusedTuning {
    int nst = 0, cyc = -1;
};
cudaError_t launch_atax_fused(const DeviceInfo &d, int64_t m, int64_t n, const float *A, const float *x,
                              float *y, void *ws, cudaStream_t s, Exch ex = Exch{}, int dst = -1, int blocks = 0,
                              FusedTuning tune = FusedTuning{});

// ---- Listing 1 in the paper's exact order (NEXT-3) ------------------------------
cudaError_t launch_partial_dot(const DeviceInfo &d, int64_t n, const float *x, const float *y, float *z, bool fma,
                               cudaStream_t s);
size_t dot_listing1_ws_bytes(int64_t n);
cudaError_t launch_dot_listing1(const DeviceInfo &d, int64_t n, const float *x, const float *y, float *result,
                                void *ws, bool fma, cudaStream_t s);

}  // namespace lift
