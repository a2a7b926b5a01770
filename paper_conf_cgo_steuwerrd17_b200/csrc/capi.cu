// capi.cu — the C ABI of include/lift.h: host-side validation, device
// configuration and dispatch to the kernels.  Validation never touches CUDA,
// so every error path is testable without a GPU.
#include <limits.h>
#include <stdio.h>
#include <string.h>

#include <initializer_list>
#include <mutex>

#include "../../include/lift.h"
#include "../../include/lift_tuning.h"
#include "../../include/lift_nvlink.h"
#include "../../include/lift_host.h"
#include "launch.h"

namespace lift {

static std::mutex g_dev_mu;
static DeviceInfo g_dev[64];

cudaError_t device_info(DeviceInfo *out) {
    int dev = 0;
    cudaError_t e = cudaGetDevice(&dev);
    if (e != cudaSuccess) return e;
    if (dev < 0 || dev >= 64) return cudaErrorInvalidDevice;
    std::lock_guard<std::mutex> lk(g_dev_mu);
    DeviceInfo &d = g_dev[dev];
    if (d.device != dev) {
        DeviceInfo t;
        t.device = dev;
        if ((e = cudaDeviceGetAttribute(&t.sms, cudaDevAttrMultiProcessorCount, dev)) != cudaSuccess) return e;
        if ((e = cudaDeviceGetAttribute(&t.smem_optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev)) != cudaSuccess)
            return e;
        if ((e = cudaDeviceGetAttribute(&t.smem_per_sm, cudaDevAttrMaxSharedMemoryPerMultiprocessor, dev)) !=
            cudaSuccess)
            return e;
        if ((e = cudaDeviceGetAttribute(&t.max_threads_sm, cudaDevAttrMaxThreadsPerMultiProcessor, dev)) !=
            cudaSuccess)
            return e;
        if ((e = cudaDeviceGetAttribute(&t.regs_per_sm, cudaDevAttrMaxRegistersPerMultiprocessor, dev)) !=
            cudaSuccess)
            return e;
        // eager load (lazy loading at a first launch waits for an idle device, which a
        // kernel spinning on a peer's flag never allows)
        if ((e = preload_dot()) != cudaSuccess || (e = preload_gemv()) != cudaSuccess ||
            (e = preload_atax()) != cudaSuccess || (e = preload_listing1()) != cudaSuccess)
            return e;
        d = t;
    }
    *out = d;
    return cudaSuccess;
}

}  // namespace lift

using lift::DeviceInfo;

static thread_local char g_cuda_err[256] = "no error";

static int cuda_status(cudaError_t e) {
    if (e == cudaSuccess) return LIFT_OK;
    snprintf(g_cuda_err, sizeof g_cuda_err, "%s: %s", cudaGetErrorName(e), cudaGetErrorString(e));
    return LIFT_ERR_CUDA;
}

// ---------------------------------------------------------------------------
// validation helpers (pure host logic)
// ---------------------------------------------------------------------------
struct Range {
    uintptr_t lo, hi;  // [lo, hi)
};
static Range rng(const void *p, uint64_t bytes) {
    uintptr_t a = reinterpret_cast<uintptr_t>(p);
    return Range{a, a + (uintptr_t)bytes};
}
static bool overlap(Range a, Range b) {
    if (a.lo == a.hi || b.lo == b.hi) return false;
    return a.lo < b.hi && b.lo < a.hi;
}
static bool mis4(const void *p) { return (reinterpret_cast<uintptr_t>(p) & 3) != 0; }

// elements m*n with 4-byte elements must be addressable in int64 bytes
static bool size_ok(int64_t m, int64_t n) {
    if (m < 0 || n < 0) return false;
    if (m == 0 || n == 0) return true;
    return m <= (INT64_MAX / 4) / n;
}

extern "C" {

size_t lift_dot_workspace_bytes(int64_t n) {
    (void)n;
    return lift::kDotTicketBytes + (size_t)lift::kDotMaxBlocks * sizeof(float);
}

int lift_dot(int64_t n, const float *x, const float *y, float *result, void *workspace, size_t workspace_bytes,
             lift_stream_t stream) {
    if (!size_ok(n, 1)) return LIFT_ERR_BAD_SIZE;
    if (result == nullptr) return LIFT_ERR_NULL_PTR;
    if (n > 0 && (x == nullptr || y == nullptr)) return LIFT_ERR_NULL_PTR;
    if (mis4(result) || (n > 0 && (mis4(x) || mis4(y)))) return LIFT_ERR_MISALIGNED;
    if (workspace == nullptr || workspace_bytes < lift_dot_workspace_bytes(n) ||
        (reinterpret_cast<uintptr_t>(workspace) & 15) != 0)
        return LIFT_ERR_WORKSPACE;
    const Range rr = rng(result, 4), rw = rng(workspace, workspace_bytes);
    const Range rx = rng(x, (uint64_t)n * 4), ry = rng(y, (uint64_t)n * 4);
    if (overlap(rr, rx) || overlap(rr, ry) || overlap(rr, rw) || overlap(rw, rx) || overlap(rw, ry))
        return LIFT_ERR_ALIAS;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    return cuda_status(lift::launch_dot(d, n, x, y, result, workspace, (cudaStream_t)stream));
}

static int check_gemv_family(int64_t m, int64_t n, const float *A, const float *B, bool two, const float *x,
                             const float *y) {
    if (!size_ok(m, n)) return LIFT_ERR_BAD_SIZE;
    if (m > 0 && y == nullptr) return LIFT_ERR_NULL_PTR;
    if (m > 0 && n > 0 && (A == nullptr || x == nullptr || (two && B == nullptr))) return LIFT_ERR_NULL_PTR;
    if (m > 0 && mis4(y)) return LIFT_ERR_MISALIGNED;
    if (m > 0 && n > 0 && (mis4(A) || mis4(x) || (two && mis4(B)))) return LIFT_ERR_MISALIGNED;
    if (m > 0) {
        const Range ry = rng(y, (uint64_t)m * 4);
        const uint64_t mat = (uint64_t)m * (uint64_t)n * 4;
        if (overlap(ry, rng(A, mat)) || overlap(ry, rng(x, (uint64_t)n * 4)) || (two && overlap(ry, rng(B, mat))))
            return LIFT_ERR_ALIAS;
    }
    return LIFT_OK;
}

int lift_gemv_tuned(int64_t m, int64_t n, const float *A, const float *x, float *y, int wpr, int rg, int blocks,
                    int xsmem, int lb, lift_stream_t stream) {
    int st = check_gemv_family(m, n, A, nullptr, false, x, y);
    if (st != LIFT_OK) return st;
    if (m == 0) return LIFT_OK;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    lift::GemvConfig cfg;
    cfg.wpr = wpr;
    cfg.rg = rg;
    cfg.blocks = blocks;
    cfg.xsmem = xsmem;
    cfg.lb = lb;
    lift::GemvArgs g;
    g.m = m;
    g.n = n;
    g.lda = n;
    g.A = A;
    g.x = x;
    g.y = y;
    return cuda_status(lift::launch_gemv(d, g, cfg, (cudaStream_t)stream));
}

int lift_gemv(int64_t m, int64_t n, const float *A, const float *x, float *y, lift_stream_t stream) {
    return lift_gemv_tuned(m, n, A, x, y, 0, 0, 0, -1, 0, stream);
}

int lift_gesummv_tuned(int64_t m, int64_t n, float alpha, const float *A, float beta, const float *B, const float *x,
                       float *y, int wpr, int rg, int blocks, int xsmem, int lb, lift_stream_t stream) {
    int st = check_gemv_family(m, n, A, B, true, x, y);
    if (st != LIFT_OK) return st;
    if (m == 0) return LIFT_OK;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    lift::GemvConfig cfg;
    cfg.wpr = wpr;
    cfg.rg = rg;
    cfg.blocks = blocks;
    cfg.xsmem = xsmem;
    cfg.lb = lb;
    lift::GemvArgs g;
    g.nmat = 2;
    g.m = m;
    g.n = n;
    g.lda = n;
    g.A = A;
    g.B = B;
    g.x = x;
    g.y = y;
    g.alpha = alpha;
    g.beta = beta;
    g.epi = lift::kEpiSum2;
    return cuda_status(lift::launch_gemv(d, g, cfg, (cudaStream_t)stream));
}

int lift_gesummv(int64_t m, int64_t n, float alpha, const float *A, float beta, const float *B, const float *x,
                 float *y, lift_stream_t stream) {
    return lift_gesummv_tuned(m, n, alpha, A, beta, B, x, y, 0, 0, 0, -1, 0, stream);
}

size_t lift_atax_workspace_bytes(int64_t m, int64_t n) {
    if (!size_ok(m, n)) return 0;
    size_t a = lift::atax_twopass_ws_bytes(m, n), b = lift::atax_fused_ws_bytes(m, n);
    return a > b ? a : b;
}

int lift_atax_algo_run(int algo, int64_t m, int64_t n, const float *A, const float *x, float *y, void *workspace,
                       size_t workspace_bytes, lift_stream_t stream) {
    if (algo < LIFT_ATAX_AUTO || algo > LIFT_ATAX_TWOPASS) return LIFT_ERR_BAD_SIZE;
    if (!size_ok(m, n)) return LIFT_ERR_BAD_SIZE;
    if (n > 0 && y == nullptr) return LIFT_ERR_NULL_PTR;
    if (m > 0 && n > 0 && (A == nullptr || x == nullptr)) return LIFT_ERR_NULL_PTR;
    if (n > 0 && mis4(y)) return LIFT_ERR_MISALIGNED;
    if (m > 0 && n > 0 && (mis4(A) || mis4(x))) return LIFT_ERR_MISALIGNED;
    if (workspace == nullptr || workspace_bytes < lift_atax_workspace_bytes(m, n) ||
        (reinterpret_cast<uintptr_t>(workspace) & 15) != 0)
        return LIFT_ERR_WORKSPACE;
    const uint64_t mat = (uint64_t)m * (uint64_t)n * 4;
    const Range ry = rng(y, (uint64_t)n * 4), rw = rng(workspace, workspace_bytes);
    const Range rA = rng(A, mat), rx = rng(x, (uint64_t)n * 4);
    if (overlap(ry, rA) || overlap(ry, rx) || overlap(ry, rw) || overlap(rw, rA) || overlap(rw, rx))
        return LIFT_ERR_ALIAS;
    const bool aligned = ((reinterpret_cast<uintptr_t>(A) | reinterpret_cast<uintptr_t>(x) |
                           reinterpret_cast<uintptr_t>(y)) & 15) == 0;
    const bool fused_ok = lift::atax_fused_supported(m, n, aligned);
    if (algo == LIFT_ATAX_FUSED && !fused_ok && m > 0 && n > 0) return LIFT_ERR_BAD_SIZE;
    if (n == 0) return LIFT_OK;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    const bool fused = (algo == LIFT_ATAX_FUSED) || (algo == LIFT_ATAX_AUTO && lift::atax_fused_preferred(m, n, aligned));
    if (fused) return cuda_status(lift::launch_atax_fused(d, m, n, A, x, y, workspace, (cudaStream_t)stream));
    return cuda_status(lift::launch_atax_twopass(d, m, n, A, x, y, workspace, (cudaStream_t)stream));
}

int lift_atax(int64_t m, int64_t n, const float *A, const float *x, float *y, void *workspace,
              size_t workspace_bytes, lift_stream_t stream) {
    return lift_atax_algo_run(LIFT_ATAX_AUTO, m, n, A, x, y, workspace, workspace_bytes, stream);
}

int lift_atax_fused_grid(int64_t m, int64_t n, int *blocks, int *cluster) {
    if (blocks == nullptr || cluster == nullptr) return LIFT_ERR_NULL_PTR;
    if (!size_ok(m, n) || !lift::atax_fused_supported(m, n, true)) return LIFT_ERR_BAD_SIZE;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    return cuda_status(lift::atax_fused_grid(d, m, n, blocks, cluster));
}

int lift_atax_fused_tuned(int64_t m, int64_t n, const float *A, const float *x, float *y, void *workspace,
                          size_t workspace_bytes, int nst, int cyclic, lift_stream_t stream) {
    // validation of lift_atax_algo_run(LIFT_ATAX_FUSED, ...), then the overrides
    if (!size_ok(m, n)) return LIFT_ERR_BAD_SIZE;
    if (n > 0 && y == nullptr) return LIFT_ERR_NULL_PTR;
    if (m > 0 && n > 0 && (A == nullptr || x == nullptr)) return LIFT_ERR_NULL_PTR;
    if (n > 0 && mis4(y)) return LIFT_ERR_MISALIGNED;
    if (m > 0 && n > 0 && (mis4(A) || mis4(x))) return LIFT_ERR_MISALIGNED;
    if (workspace == nullptr || workspace_bytes < lift_atax_workspace_bytes(m, n) ||
        (reinterpret_cast<uintptr_t>(workspace) & 15) != 0)
        return LIFT_ERR_WORKSPACE;
    const uint64_t mat = (uint64_t)m * (uint64_t)n * 4;
    const Range ry = rng(y, (uint64_t)n * 4), rw = rng(workspace, workspace_bytes);
    const Range rA = rng(A, mat), rx = rng(x, (uint64_t)n * 4);
    if (overlap(ry, rA) || overlap(ry, rx) || overlap(ry, rw) || overlap(rw, rA) || overlap(rw, rx))
        return LIFT_ERR_ALIAS;
    const bool aligned = ((reinterpret_cast<uintptr_t>(A) | reinterpret_cast<uintptr_t>(x) |
                           reinterpret_cast<uintptr_t>(y)) & 15) == 0;
    if (m > 0 && n > 0 && !lift::atax_fused_supported(m, n, aligned)) return LIFT_ERR_BAD_SIZE;
    if (n == 0) return LIFT_OK;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    lift::FusedTuning t;
    t.nst = nst;
    t.cyc = cyclic;
    return cuda_status(
        lift::launch_atax_fused(d, m, n, A, x, y, workspace, (cudaStream_t)stream, lift::Exch{}, -1, 0, t));
}

// (layout, trans) -> does the row-major kernel walk rows of the stored matrix (false)
// or its columns (true)?  Column-major A is the row-major A^T.
static bool sgemv_colpath(int layout, int trans) { return (layout == 0) == (trans == 1); }

size_t lift_sgemv_workspace_bytes(int layout, int trans, int64_t m, int64_t n) {
    if (!size_ok(m, n) || (layout != 0 && layout != 1) || (trans != 0 && trans != 1)) return 0;
    if (!sgemv_colpath(layout, trans)) return 0;
    // stored row-major matrix R = (layout 0 ? A : A^T): rows x cols; the column path reduces over rows
    const int64_t cols = layout == 0 ? n : m;
    const int64_t rows = layout == 0 ? m : n;
    return lift::gemv_t_ws_bytes(rows, cols);
}

int lift_sgemv(int layout, int trans, int64_t m, int64_t n, float alpha, const float *A, int64_t lda, const float *x,
               float beta, float *y, void *workspace, size_t workspace_bytes, lift_stream_t stream) {
    if ((layout != 0 && layout != 1) || (trans != 0 && trans != 1)) return LIFT_ERR_BAD_SIZE;
    if (!size_ok(m, n)) return LIFT_ERR_BAD_SIZE;
    // the stored matrix as row-major R: rows x cols with row stride lda
    const int64_t rows = layout == 0 ? m : n, cols = layout == 0 ? n : m;
    if (lda < (cols > 1 ? cols : 1)) return LIFT_ERR_BAD_SIZE;
    if (rows > 0 && !size_ok(rows, lda)) return LIFT_ERR_BAD_SIZE;
    const int64_t xlen = trans == 0 ? n : m, ylen = trans == 0 ? m : n;
    if (ylen > 0 && y == nullptr) return LIFT_ERR_NULL_PTR;
    if (m > 0 && n > 0 && (A == nullptr || x == nullptr)) return LIFT_ERR_NULL_PTR;
    if (ylen > 0 && mis4(y)) return LIFT_ERR_MISALIGNED;
    if (m > 0 && n > 0 && (mis4(A) || mis4(x))) return LIFT_ERR_MISALIGNED;
    const bool colpath = sgemv_colpath(layout, trans);
    const size_t need = lift_sgemv_workspace_bytes(layout, trans, m, n);
    if (need > 0 && (workspace == nullptr || workspace_bytes < need || (reinterpret_cast<uintptr_t>(workspace) & 15)))
        return LIFT_ERR_WORKSPACE;
    if (ylen > 0) {
        const uint64_t abytes = rows > 0 ? ((uint64_t)(rows - 1) * (uint64_t)lda + (uint64_t)cols) * 4 : 0;
        const Range ry = rng(y, (uint64_t)ylen * 4);
        if (overlap(ry, rng(A, abytes)) || overlap(ry, rng(x, (uint64_t)xlen * 4)) ||
            (need > 0 && overlap(ry, rng(workspace, workspace_bytes))))
            return LIFT_ERR_ALIAS;
        if (need > 0 && (overlap(rng(workspace, workspace_bytes), rng(A, abytes)) ||
                         overlap(rng(workspace, workspace_bytes), rng(x, (uint64_t)xlen * 4))))
            return LIFT_ERR_ALIAS;
    }
    if (ylen == 0) return LIFT_OK;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    if (colpath)  // y (length cols) = alpha * R^T x + beta * y
        return cuda_status(lift::launch_gemv_t(d, rows, cols, lda, alpha, A, x, beta, y, workspace,
                                               (cudaStream_t)stream));
    lift::GemvArgs g;  // y (length rows) = alpha * R x + beta * y
    g.m = rows;
    g.n = cols;
    g.lda = lda;
    g.A = A;
    g.x = x;
    g.y = y;
    g.alpha = alpha;
    g.beta = beta;
    g.epi = lift::kEpiAxpby;
    return cuda_status(lift::launch_gemv(d, g, lift::GemvConfig{}, (cudaStream_t)stream));
}

int lift_partial_dot(int64_t n, const float *x, const float *y, float *z, int contract, lift_stream_t stream) {
    if (!size_ok(n, 1)) return LIFT_ERR_BAD_SIZE;
    if (contract != 0 && contract != 1) return LIFT_ERR_BAD_SIZE;
    const int64_t groups = n / 128;
    if (groups == 0) return LIFT_OK;
    if (x == nullptr || y == nullptr || z == nullptr) return LIFT_ERR_NULL_PTR;
    if (mis4(x) || mis4(y) || mis4(z)) return LIFT_ERR_MISALIGNED;
    const Range rz = rng(z, (uint64_t)groups * 4);
    if (overlap(rz, rng(x, (uint64_t)n * 4)) || overlap(rz, rng(y, (uint64_t)n * 4))) return LIFT_ERR_ALIAS;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    return cuda_status(lift::launch_partial_dot(d, n, x, y, z, contract == 1, (cudaStream_t)stream));
}

size_t lift_dot_listing1_workspace_bytes(int64_t n) {
    if (!size_ok(n, 1)) return 0;
    return lift::dot_listing1_ws_bytes(n);
}

int lift_dot_listing1(int64_t n, const float *x, const float *y, float *result, void *workspace,
                      size_t workspace_bytes, int contract, lift_stream_t stream) {
    if (!size_ok(n, 1)) return LIFT_ERR_BAD_SIZE;
    if (contract != 0 && contract != 1) return LIFT_ERR_BAD_SIZE;
    if (result == nullptr) return LIFT_ERR_NULL_PTR;
    if (n > 0 && (x == nullptr || y == nullptr)) return LIFT_ERR_NULL_PTR;
    if (mis4(result) || (n > 0 && (mis4(x) || mis4(y)))) return LIFT_ERR_MISALIGNED;
    if (workspace == nullptr || workspace_bytes < lift::dot_listing1_ws_bytes(n) ||
        (reinterpret_cast<uintptr_t>(workspace) & 15) != 0)
        return LIFT_ERR_WORKSPACE;
    const Range rr = rng(result, 4), rw = rng(workspace, workspace_bytes);
    const Range rx = rng(x, (uint64_t)n * 4), ry = rng(y, (uint64_t)n * 4);
    if (overlap(rr, rx) || overlap(rr, ry) || overlap(rr, rw) || overlap(rw, rx) || overlap(rw, ry))
        return LIFT_ERR_ALIAS;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    return cuda_status(
        lift::launch_dot_listing1(d, n, x, y, result, workspace, contract == 1, (cudaStream_t)stream));
}

// ---------------------------------------------------------------------------
// collectives fused into the kernels (NEXT-2)
// ---------------------------------------------------------------------------
static int64_t exch_cap(int kind, int64_t len, int world) {
    if (kind == LIFT_EXCH_DOT) return lift::kMaxWorld;
    if (kind == LIFT_EXCH_GATHER) return len;
    return (int64_t)world * len;
}

size_t lift_exchange_bytes(int kind, int64_t len, int world) {
    if (kind < LIFT_EXCH_DOT || kind > LIFT_EXCH_REDUCE || world < 1 || world > lift::kMaxWorld || len < 0)
        return 0;
    if (!size_ok(exch_cap(kind, len, world), 2)) return 0;
    const size_t b = lift::kExchHeader + 2 * (size_t)exch_cap(kind, len, world) * sizeof(float);
    return (b + 255) / 256 * 256;
}

static int check_group(void *const *peers, int rank, int world) {
    if (world < 1 || world > lift::kMaxWorld || rank < 0 || rank >= world) return LIFT_ERR_BAD_SIZE;
    if (peers == nullptr) return LIFT_ERR_NULL_PTR;
    if ((reinterpret_cast<uintptr_t>(peers) & 7) != 0) return LIFT_ERR_MISALIGNED;
    return LIFT_OK;
}

static lift::Exch make_exch(void *const *peers, int rank, int world, int64_t cap) {
    lift::Exch e;
    e.peers = reinterpret_cast<char *const *>(peers);
    e.rank = rank;
    e.world = world;
    e.cap = cap;
    return e;
}

int lift_dot_allreduce(int64_t n, const float *x, const float *y, float *result, void *workspace,
                       size_t workspace_bytes, void *const *peers, int rank, int world,
                       lift_stream_t stream) {
    int st = check_group(peers, rank, world);
    if (st != LIFT_OK) return st;
    if (!size_ok(n, 1)) return LIFT_ERR_BAD_SIZE;
    if (result == nullptr) return LIFT_ERR_NULL_PTR;
    if (n > 0 && (x == nullptr || y == nullptr)) return LIFT_ERR_NULL_PTR;
    if (mis4(result) || (n > 0 && (mis4(x) || mis4(y)))) return LIFT_ERR_MISALIGNED;
    if (workspace == nullptr || workspace_bytes < lift_dot_workspace_bytes(n) ||
        (reinterpret_cast<uintptr_t>(workspace) & 15) != 0)
        return LIFT_ERR_WORKSPACE;
    const Range rr = rng(result, 4), rw = rng(workspace, workspace_bytes);
    const Range rx = rng(x, (uint64_t)n * 4), ry = rng(y, (uint64_t)n * 4);
    if (overlap(rr, rx) || overlap(rr, ry) || overlap(rr, rw) || overlap(rw, rx) || overlap(rw, ry))
        return LIFT_ERR_ALIAS;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    return cuda_status(lift::launch_dot(d, n, x, y, result, workspace, (cudaStream_t)stream,
                                        make_exch(peers, rank, world, lift::kMaxWorld)));
}

static int gather_common(int nmat, int64_t m, int64_t n, float alpha, const float *A, float beta, const float *B,
                         const float *x, int64_t row0, int64_t m_total, float *y, void *workspace,
                         size_t workspace_bytes, void *const *peers, int rank, int world,
                         lift_stream_t stream) {
    int st = check_group(peers, rank, world);
    if (st != LIFT_OK) return st;
    if (!size_ok(m, n) || !size_ok(m_total, 1) || row0 < 0 || row0 + m > m_total) return LIFT_ERR_BAD_SIZE;
    if (m_total > 0 && y == nullptr) return LIFT_ERR_NULL_PTR;
    if (m > 0 && n > 0 && (A == nullptr || x == nullptr || (nmat == 2 && B == nullptr))) return LIFT_ERR_NULL_PTR;
    if ((m_total > 0 && mis4(y)) || (m > 0 && n > 0 && (mis4(A) || mis4(x) || (nmat == 2 && mis4(B)))))
        return LIFT_ERR_MISALIGNED;
    if (workspace == nullptr || workspace_bytes < 16 || (reinterpret_cast<uintptr_t>(workspace) & 15) != 0)
        return LIFT_ERR_WORKSPACE;
    const Range ry = rng(y, (uint64_t)m_total * 4), rw = rng(workspace, workspace_bytes);
    const uint64_t mat = (uint64_t)m * (uint64_t)n * 4;
    if (overlap(ry, rng(A, mat)) || overlap(ry, rng(x, (uint64_t)n * 4)) || (nmat == 2 && overlap(ry, rng(B, mat))) ||
        overlap(ry, rw))
        return LIFT_ERR_ALIAS;
    // the ticket is written by the kernel: it must not live inside an input either
    if (overlap(rw, rng(A, mat)) || overlap(rw, rng(x, (uint64_t)n * 4)) || (nmat == 2 && overlap(rw, rng(B, mat))))
        return LIFT_ERR_ALIAS;
    if (m_total == 0) return LIFT_OK;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    lift::GemvArgs g;
    g.nmat = nmat;
    g.m = m;
    g.n = n;
    g.lda = n;
    g.A = A;
    g.B = B;
    g.x = x;
    g.y = y;
    g.alpha = alpha;
    g.beta = beta;
    g.epi = nmat == 2 ? lift::kEpiSum2 : lift::kEpiStore;
    g.ex = make_exch(peers, rank, world, m_total);
    g.row0 = row0;
    g.m_total = m_total;
    g.ticket = static_cast<unsigned int *>(workspace);
    return cuda_status(lift::launch_gemv(d, g, lift::GemvConfig{}, (cudaStream_t)stream));
}

int lift_gemv_allgather(int64_t m, int64_t n, const float *A, const float *x, int64_t row0, int64_t m_total,
                        float *y, void *workspace, size_t workspace_bytes, void *const *peers, int rank, int world,
                        lift_stream_t stream) {
    return gather_common(1, m, n, 1.f, A, 0.f, nullptr, x, row0, m_total, y, workspace, workspace_bytes, peers, rank,
                         world, stream);
}

int lift_gesummv_allgather(int64_t m, int64_t n, float alpha, const float *A, float beta, const float *B,
                           const float *x, int64_t row0, int64_t m_total, float *y, void *workspace,
                           size_t workspace_bytes, void *const *peers, int rank, int world,
                           lift_stream_t stream) {
    return gather_common(2, m, n, alpha, A, beta, B, x, row0, m_total, y, workspace, workspace_bytes, peers, rank,
                         world, stream);
}

int lift_atax_reduce(int64_t m, int64_t n, const float *A, const float *x, float *y, void *workspace,
                     size_t workspace_bytes, void *const *peers, int rank, int world, int dst,
                     int blocks, lift_stream_t stream) {
    int st = check_group(peers, rank, world);
    if (st != LIFT_OK) return st;
    if (dst < -1 || dst >= world || blocks < 0) return LIFT_ERR_BAD_SIZE;
    if (!size_ok(m, n)) return LIFT_ERR_BAD_SIZE;
    if (n > 0 && (y == nullptr || x == nullptr || (m > 0 && A == nullptr))) return LIFT_ERR_NULL_PTR;
    if (n > 0 && (mis4(y) || mis4(x) || (m > 0 && mis4(A)))) return LIFT_ERR_MISALIGNED;
    // 4-byte aligned but not 16: an unsupported shape for the fused kernel (as lift_atax FUSED)
    const bool aligned = ((reinterpret_cast<uintptr_t>(A) | reinterpret_cast<uintptr_t>(x) |
                           reinterpret_cast<uintptr_t>(y)) & 15) == 0;
    if (n > 0 && !lift::atax_fused_exchange_supported(m > 0 ? m : 1, n, aligned)) return LIFT_ERR_BAD_SIZE;
    if (workspace == nullptr || workspace_bytes < lift_atax_workspace_bytes(m, n) ||
        (reinterpret_cast<uintptr_t>(workspace) & 15) != 0)
        return LIFT_ERR_WORKSPACE;
    const uint64_t mat = (uint64_t)m * (uint64_t)n * 4;
    const Range ry = rng(y, (uint64_t)n * 4), rw = rng(workspace, workspace_bytes);
    const Range rA = rng(A, mat), rx = rng(x, (uint64_t)n * 4);
    if (overlap(ry, rA) || overlap(ry, rx) || overlap(ry, rw) || overlap(rw, rA) || overlap(rw, rx))
        return LIFT_ERR_ALIAS;
    if (n == 0) return LIFT_OK;
    DeviceInfo d;
    cudaError_t e = lift::device_info(&d);
    if (e != cudaSuccess) return cuda_status(e);
    return cuda_status(lift::launch_atax_fused(d, m, n, A, x, y, workspace, (cudaStream_t)stream,
                                               make_exch(peers, rank, world, (int64_t)world * n), dst,
                                               blocks));
}

// ---------------------------------------------------------------------------
// end to end from host buffers (lift_host.h)
// ---------------------------------------------------------------------------
static int h2d(void *dev, const void *host, uint64_t bytes, lift_stream_t stream) {
    if (bytes == 0) return LIFT_OK;
    return cuda_status(cudaMemcpyAsync(dev, host, bytes, cudaMemcpyHostToDevice, (cudaStream_t)stream));
}
static int d2h(void *host, const void *dev, uint64_t bytes, lift_stream_t stream) {
    if (bytes == 0) return LIFT_OK;
    return cuda_status(cudaMemcpyAsync(host, dev, bytes, cudaMemcpyDeviceToHost, (cudaStream_t)stream));
}
static bool any_overlap(std::initializer_list<Range> rs) {
    const Range *v = rs.begin();
    const size_t k = rs.size();
    for (size_t i = 0; i < k; ++i)
        for (size_t j = i + 1; j < k; ++j)
            if (overlap(v[i], v[j])) return true;
    return false;
}

int lift_dot_host(int64_t n, const float *x_host, const float *y_host, float *result_host, float *x_dev, float *y_dev,
                  float *result_dev, void *workspace, size_t workspace_bytes, lift_stream_t stream) {
    if (!size_ok(n, 1)) return LIFT_ERR_BAD_SIZE;
    if (result_host == nullptr || (n > 0 && (x_host == nullptr || y_host == nullptr))) return LIFT_ERR_NULL_PTR;
    const uint64_t b = (uint64_t)n * 4;
    if (x_dev && y_dev && result_dev &&
        any_overlap({rng(x_dev, b), rng(y_dev, b), rng(result_dev, 4), rng(workspace, workspace_bytes)}))
        return LIFT_ERR_ALIAS;
    int st;
    if ((st = h2d(x_dev, x_host, b, stream)) || (st = h2d(y_dev, y_host, b, stream))) return st;
    if ((st = lift_dot(n, x_dev, y_dev, result_dev, workspace, workspace_bytes, stream))) return st;
    return d2h(result_host, result_dev, 4, stream);
}

int lift_gemv_host(int64_t m, int64_t n, const float *A_host, const float *x_host, float *y_host, float *A_dev,
                   float *x_dev, float *y_dev, lift_stream_t stream) {
    if (!size_ok(m, n)) return LIFT_ERR_BAD_SIZE;
    if (m > 0 && (y_host == nullptr || (n > 0 && (A_host == nullptr || x_host == nullptr)))) return LIFT_ERR_NULL_PTR;
    const uint64_t ba = (uint64_t)m * (uint64_t)n * 4, bx = (uint64_t)n * 4, by = (uint64_t)m * 4;
    if (any_overlap({rng(A_dev, ba), rng(x_dev, bx), rng(y_dev, by)})) return LIFT_ERR_ALIAS;
    if (m == 0) return LIFT_OK;
    int st;
    if ((st = h2d(A_dev, A_host, ba, stream)) || (st = h2d(x_dev, x_host, bx, stream))) return st;
    if ((st = lift_gemv(m, n, A_dev, x_dev, y_dev, stream))) return st;
    return d2h(y_host, y_dev, by, stream);
}

int lift_gesummv_host(int64_t m, int64_t n, float alpha, const float *A_host, float beta, const float *B_host,
                      const float *x_host, float *y_host, float *A_dev, float *B_dev, float *x_dev, float *y_dev,
                      lift_stream_t stream) {
    if (!size_ok(m, n)) return LIFT_ERR_BAD_SIZE;
    if (m > 0 && (y_host == nullptr || (n > 0 && (A_host == nullptr || B_host == nullptr || x_host == nullptr))))
        return LIFT_ERR_NULL_PTR;
    const uint64_t ba = (uint64_t)m * (uint64_t)n * 4, bx = (uint64_t)n * 4, by = (uint64_t)m * 4;
    if (any_overlap({rng(A_dev, ba), rng(B_dev, ba), rng(x_dev, bx), rng(y_dev, by)})) return LIFT_ERR_ALIAS;
    if (m == 0) return LIFT_OK;
    int st;
    if ((st = h2d(A_dev, A_host, ba, stream)) || (st = h2d(B_dev, B_host, ba, stream)) ||
        (st = h2d(x_dev, x_host, bx, stream)))
        return st;
    if ((st = lift_gesummv(m, n, alpha, A_dev, beta, B_dev, x_dev, y_dev, stream))) return st;
    return d2h(y_host, y_dev, by, stream);
}

int lift_atax_host(int64_t m, int64_t n, const float *A_host, const float *x_host, float *y_host, float *A_dev,
                   float *x_dev, float *y_dev, void *workspace, size_t workspace_bytes, lift_stream_t stream) {
    if (!size_ok(m, n)) return LIFT_ERR_BAD_SIZE;
    if (n > 0 && (y_host == nullptr || (m > 0 && (A_host == nullptr || x_host == nullptr)))) return LIFT_ERR_NULL_PTR;
    const uint64_t ba = (uint64_t)m * (uint64_t)n * 4, bx = (uint64_t)n * 4;
    if (any_overlap({rng(A_dev, ba), rng(x_dev, bx), rng(y_dev, bx), rng(workspace, workspace_bytes)}))
        return LIFT_ERR_ALIAS;
    if (n == 0) return LIFT_OK;
    int st;
    if ((st = h2d(A_dev, A_host, ba, stream)) || (st = h2d(x_dev, x_host, bx, stream))) return st;
    if ((st = lift_atax(m, n, A_dev, x_dev, y_dev, workspace, workspace_bytes, stream))) return st;
    return d2h(y_host, y_dev, bx, stream);
}

const char *lift_strerror(int status) {
    switch (status) {
        case LIFT_OK: return "LIFT_OK: success";
        case LIFT_ERR_NULL_PTR: return "LIFT_ERR_NULL_PTR: a required pointer is NULL";
        case LIFT_ERR_BAD_SIZE: return "LIFT_ERR_BAD_SIZE: negative or overflowing size, or unsupported shape";
        case LIFT_ERR_MISALIGNED: return "LIFT_ERR_MISALIGNED: pointer not 4-byte aligned";
        case LIFT_ERR_ALIAS: return "LIFT_ERR_ALIAS: output overlaps an input or the workspace";
        case LIFT_ERR_WORKSPACE: return "LIFT_ERR_WORKSPACE: workspace NULL, too small or not 16-byte aligned";
        case LIFT_ERR_CUDA: return "LIFT_ERR_CUDA: CUDA launch error (see lift_last_cuda_error)";
        default: return "unknown lift status";
    }
}

const char *lift_last_cuda_error(void) { return g_cuda_err; }

int lift_version(void) { return (2 << 16) | 0; }

}  // extern "C"
