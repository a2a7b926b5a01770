// gemv.cu — k_gemv: GEMV y = A x and GESUMMV y = alpha A x + beta B x
// (Table 1), the zip -> map(x) -> reduce(+) kernel
// applied per row with x reused across rows.
//
// Mapping of the Lift patterns onto sm_100a:
//   mapWrg over rows (L359-367)     persistent grid-stride loop over row groups
//   toLocal(x) (L368-377)           x staged ONCE per block into smem by the
//                                   bulk-copy engine (cp.async.bulk + mbarrier,
//                                   SASS UBLKCP), overlapped with the first A loads
//   zip(A_i, x) / asVector4          128-bit streaming loads of A (no L1 alloc)
//   reduceSeq(multAndSumUp) (L320)   per-lane FMA fold in registers
//   iterate tree (L394-397)          warp butterfly + fixed pairwise tree
//   GESUMMV's zip of (A_i, B_i)      two accumulator sets, one pass, y_i =
//                                    alpha*sA + beta*sB: Ax and Bx never exist
//
// Canonical per-row order (independent of m, of the launch configuration and
// of row sharding): a row of nv = n/VEC vectors is cut into 8 "slices" of
// 32 virtual lanes.  Virtual lane v = 32*p + l (slice p, lane l) folds the
// vectors j = v, v + 256, v + 512, ... in increasing j into one accumulator
// (per component for float4), starting from 0.  Each virtual lane's value is
// (acc.x + acc.y) + (acc.z + acc.w); each slice is a 32-lane butterfly; the
// row is the pairwise tree over the 8 slices.  A block row group of WPR warps
// computes 8/WPR slices per warp, so every WPR gives the same bits.
#include "common.cuh"
#include "exchange.cuh"
#include "launch.h"

namespace lift {

// L2 prefetch before griddepcontrol.wait (see k_gemv): rows per first-wave row group,
// bytes per row, and whether GESUMMV also prefetches B (-D overrides for A/B builds)
#ifndef LIFT_GEMV_PF_BYTES
#define LIFT_GEMV_PF_BYTES 16384
#endif
#ifndef LIFT_GEMV_PF_ROWS
#define LIFT_GEMV_PF_ROWS 1
#endif
#ifndef LIFT_GESUMMV_PF_BYTES
#define LIFT_GESUMMV_PF_BYTES LIFT_GEMV_PF_BYTES
#endif
// GESUMMV prefetches A's row only: back to back 4096^2 19.9 us vs 20.2 with A and B,
// 20.8 with none; launched alone all within noise (profiles/r02_gesummv_prefetch_ab.txt)
#ifndef LIFT_GESUMMV_PF_B
#define LIFT_GESUMMV_PF_B 0
#endif
constexpr int kPfRows = LIFT_GEMV_PF_ROWS;
constexpr int64_t kPfBytes = LIFT_GEMV_PF_BYTES, kPfBytesGesummv = LIFT_GESUMMV_PF_BYTES;
constexpr bool kPfGesummvB = LIFT_GESUMMV_PF_B != 0;

constexpr int kSlices = 8;
constexpr int kVLanes = kSlices * kWarp;  // 256 virtual lanes per row

template <int VEC>
struct Vec;
template <>
struct Vec<4> {
    using T = float4;
    static __device__ __forceinline__ T zero() { return zero4(); }
    static __device__ __forceinline__ T ld_stream(const T *p) { return ld_stream4(p); }
    static __device__ __forceinline__ T ld_x_smem(const T *p) { return *p; }
    static __device__ __forceinline__ T ld_x_global(const T *p) { return ld_ro4(p); }
    static __device__ __forceinline__ void fma(T &acc, T a, T b) { fma4(acc, a, b); }
    static __device__ __forceinline__ float hsum(T v) { return hsum4(v); }
};
template <>
struct Vec<1> {
    using T = float;
    static __device__ __forceinline__ T zero() { return 0.f; }
    static __device__ __forceinline__ T ld_stream(const T *p) { return ld_stream1(p); }
    static __device__ __forceinline__ T ld_x_smem(const T *p) { return *p; }
    static __device__ __forceinline__ T ld_x_global(const T *p) { return ld_ro1(p); }
    static __device__ __forceinline__ void fma(T &acc, T a, T b) { acc = __fmaf_rn(a, b, acc); }
    static __device__ __forceinline__ float hsum(T v) { return v; }
};

// smem layout: [mbarrier 16 B][red: 2 buffers x RG x NMAT x 8 floats][x: n floats, 16-B aligned]
template <int NMAT, int RG>
__host__ __device__ constexpr int gemv_red_bytes() {
    return 2 * RG * NMAT * kSlices * 4;
}
template <int NMAT, int RG>
__host__ __device__ constexpr int gemv_x_offset() {
    return (16 + gemv_red_bytes<NMAT, RG>() + 15) / 16 * 16;
}

template <int NMAT, int VEC, int WPR, int RG, bool XSMEM, int LB>
__global__ void __launch_bounds__(RG *WPR *kWarp) k_gemv(int64_t m, int64_t n, int64_t lda,
                                                        const float *__restrict__ A, const float *__restrict__ B,
                                                        const float *__restrict__ x, float *__restrict__ y,
                                                        float alpha, float beta, int epi, Exch ex, int64_t row0,
                                                        int64_t m_total, unsigned int *ticket, int pf_blocks) {
    using V = Vec<VEC>;
    using T = typename V::T;
    constexpr int KQ = kSlices / WPR;                                 // slices per warp
    constexpr int UK = (LB / (KQ * NMAT)) > 0 ? (LB / (KQ * NMAT)) : 1;  // k-steps per batch
    extern __shared__ __align__(16) unsigned char smem[];
    uint64_t *bar = reinterpret_cast<uint64_t *>(smem);
    float *red = reinterpret_cast<float *>(smem + 16);
    float *xs = reinterpret_cast<float *>(smem + gemv_x_offset<NMAT, RG>());

    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int g = warp / WPR;   // row group inside the block
    const int wr = warp % WPR;  // warp rank inside the row group
    if constexpr (VEC == 4 && LIFT_PDL_PREFETCH) {
        // the first resident wave's first row per row group (A and B are never written
        // by this kernel), up to 16 KiB of it, into L2 while the previous kernel drains
        // (common.cuh).  Later waves start beside running blocks, not after a
        // predecessor: nothing to hide there.  Same-box A/B: back to back, GEMV 4096^2
        // 10.5 us with one row, 9.9 with two, 10.1 with four, 64 KiB of one row no
        // better than 16 KiB (profiles/r02_pdl_prefetch_depth_ab.txt); launched alone
        // (no predecessor, ncu) one row is free and two cost 0.8 us
        // (profiles/r02_pdl_prefetch_isolated_ncu.txt): one row.
        if ((int)blockIdx.x < pf_blocks && wr == 0 && lane < kPfRows && n > 0) {
            const int64_t r = (int64_t)blockIdx.x * RG + g + (int64_t)lane * gridDim.x * RG;
            constexpr int64_t cap = NMAT == 2 ? kPfBytesGesummv : kPfBytes;
            const uint32_t bytes = (uint32_t)(n * 4 < cap ? n * 4 : cap);
            if (r < m && bytes > 0) {
                bulk_prefetch_l2(A + r * lda, bytes);
                if constexpr (NMAT == 2 && kPfGesummvB) bulk_prefetch_l2(B + r * lda, bytes);
            }
        }
    }
    pdl_wait();
    if (ex.world == 0) pdl_release();  // a fused collective lets nothing start early beside it
    const int64_t nv = n / VEC;
    const int64_t kcount = (nv + kVLanes - 1) / kVLanes;  // k-steps per row
    const int64_t kfull = nv / kVLanes;                   // k-steps whose every vector is in the row
    const int lane_off = kWarp * (wr * KQ) + lane;        // first virtual lane of this lane, slice q adds 32*q

    // fused all-gather: this call's epoch (its parity buffer is free: the previous
    // call's exch_finish saw every destination done with it).  The exchange stays
    // a runtime branch of the one kernel: a separate template instantiation
    // without it compiled the plain GEMV 9 % slower (profiles/r02_fused_epilogue_ab.txt).
    uint64_t ep = 0;
    if (ex.world > 0) ep = exch_epoch(ex);
    bool x_pending = false;
    if constexpr (XSMEM) {
        stage_issue(xs, x, (uint32_t)(n * 4), bar);  // toLocal(x), one bulk copy per block
        x_pending = true;
    }
    const T *xl = reinterpret_cast<const T *>(XSMEM ? xs : x) + lane_off;

    const int64_t row_step = (int64_t)gridDim.x * RG;
    int64_t row = (int64_t)blockIdx.x * RG + g;

    // One continuous stream of load batches over (row, k0): batch i+1 is
    // issued before batch i is consumed, including across the row boundary,
    // so a warp keeps loads in flight while it reduces a finished row.
    // Full batches use compile-time offsets and no predicates.
    auto load_batch = [&](int64_t r, int64_t k0, T (&dst)[NMAT][UK][KQ]) {
        const T *Ar = reinterpret_cast<const T *>(A + r * lda) + (kVLanes * k0 + lane_off);
        const T *Br = (NMAT == 2) ? reinterpret_cast<const T *>(B + r * lda) + (kVLanes * k0 + lane_off) : nullptr;
        if (k0 + UK <= kfull) {
#pragma unroll
            for (int u = 0; u < UK; ++u)
#pragma unroll
                for (int q = 0; q < KQ; ++q)
#pragma unroll
                    for (int mt = 0; mt < NMAT; ++mt)
                        dst[mt][u][q] = V::ld_stream((mt == 0 ? Ar : Br) + (kVLanes * u + kWarp * q));
        } else {
#pragma unroll
            for (int u = 0; u < UK; ++u)
#pragma unroll
                for (int q = 0; q < KQ; ++q) {
                    const bool ok = kVLanes * (k0 + u) + kWarp * q + lane_off < nv;
#pragma unroll
                    for (int mt = 0; mt < NMAT; ++mt)
                        dst[mt][u][q] = ok ? V::ld_stream((mt == 0 ? Ar : Br) + (kVLanes * u + kWarp * q)) : V::zero();
                }
        }
    };

    if (row < m) {
        T cur[NMAT][UK][KQ];
        T acc[NMAT][KQ];
#pragma unroll
        for (int mt = 0; mt < NMAT; ++mt)
#pragma unroll
            for (int q = 0; q < KQ; ++q) acc[mt][q] = V::zero();
        load_batch(row, 0, cur);
        int64_t k0 = 0;
        int buf = 0;
        while (true) {
            int64_t nk = k0 + UK, nrow = row;
            if (nk >= kcount) {
                nk = 0;
                nrow = row + row_step;
            }
            T nxt[NMAT][UK][KQ];
            if (nrow < m) load_batch(nrow, nk, nxt);
            if constexpr (XSMEM) {
                if (x_pending) {  // A loads are in flight; now wait for x
                    stage_wait(bar);
                    x_pending = false;
                }
            }
            const T *xb = xl + kVLanes * k0;
            if (k0 + UK <= kfull) {
#pragma unroll
                for (int u = 0; u < UK; ++u)
#pragma unroll
                    for (int q = 0; q < KQ; ++q) {
                        const T xv = XSMEM ? V::ld_x_smem(xb + kVLanes * u + kWarp * q)
                                           : V::ld_x_global(xb + kVLanes * u + kWarp * q);
#pragma unroll
                        for (int mt = 0; mt < NMAT; ++mt) V::fma(acc[mt][q], cur[mt][u][q], xv);
                    }
            } else {
#pragma unroll
                for (int u = 0; u < UK; ++u)
#pragma unroll
                    for (int q = 0; q < KQ; ++q) {
                        T xv = V::zero();
                        if (kVLanes * (k0 + u) + kWarp * q + lane_off < nv)
                            xv = XSMEM ? V::ld_x_smem(xb + kVLanes * u + kWarp * q)
                                       : V::ld_x_global(xb + kVLanes * u + kWarp * q);
#pragma unroll
                        for (int mt = 0; mt < NMAT; ++mt) V::fma(acc[mt][q], cur[mt][u][q], xv);
                    }
            }

            if (nk == 0) {
                // row done: slice values (butterfly), then the pairwise tree over the 8 slices
                float w[NMAT][KQ];
#pragma unroll
                for (int mt = 0; mt < NMAT; ++mt)
#pragma unroll
                    for (int q = 0; q < KQ; ++q) {
                        w[mt][q] = warp_sum(V::hsum(acc[mt][q]));
                        acc[mt][q] = V::zero();
                    }
                float s[NMAT];
                bool writer;
                if constexpr (WPR == 1) {
#pragma unroll
                    for (int mt = 0; mt < NMAT; ++mt) s[mt] = pair_tree<kSlices>(w[mt]);
                    writer = (lane == 0);
                } else {
                    float *r = red + ((buf * RG + g) * NMAT) * kSlices;
                    if (lane == 0) {
#pragma unroll
                        for (int mt = 0; mt < NMAT; ++mt)
#pragma unroll
                            for (int q = 0; q < KQ; ++q) r[mt * kSlices + wr * KQ + q] = w[mt][q];
                    }
                    if constexpr (RG == 1)
                        __syncthreads();
                    else
                        named_bar_sync(1 + g, WPR * kWarp);
                    writer = (wr == 0 && lane == 0);
                    if (writer) {
#pragma unroll
                        for (int mt = 0; mt < NMAT; ++mt) {
                            float v[kSlices];
#pragma unroll
                            for (int p = 0; p < kSlices; ++p) v[p] = r[mt * kSlices + p];
                            s[mt] = pair_tree<kSlices>(v);
                        }
                    }
                    buf ^= 1;
                }
                if (writer) {
                    float val;
                    if constexpr (NMAT == 1) {
                        if (epi == kEpiStore)
                            val = s[0];
                        else  // kEpiAxpby (BLAS: y is not read when beta == 0)
                            val = beta == 0.f ? __fmul_rn(alpha, s[0])
                                              : __fadd_rn(__fmul_rn(alpha, s[0]), __fmul_rn(beta, y[row]));
                    } else {
                        val = __fadd_rn(__fmul_rn(alpha, s[0]), __fmul_rn(beta, s[1]));
                    }
                    if (ex.world == 0) {
                        y[row] = val;
                    } else {  // fused all-gather (NEXT-2): the row goes straight to every rank
                        for (int q = 0; q < ex.world; ++q) exch_data(ex.peers[q], ex, ep)[row0 + row] = val;
                    }
                }
                if (nrow >= m) break;
            }
            row = nrow;
            k0 = nk;
#pragma unroll
            for (int mt = 0; mt < NMAT; ++mt)
#pragma unroll
                for (int u = 0; u < UK; ++u)
#pragma unroll
                    for (int q = 0; q < KQ; ++q) cur[mt][u][q] = nxt[mt][u][q];
        }
    }
    if constexpr (XSMEM) {
        // a row group that received no row must still retire the bulk copy
        if (x_pending) stage_wait(bar);
    }
    if (ex.world > 0) {
        // all-gather completion: the last block of this rank publishes to every rank,
        // waits for every rank, then copies the gathered y out of the exchange area
        __shared__ int am_last;
        __syncthreads();
        if (threadIdx.x == 0)  // gpu-scope release of this block's row stores; the last block
            // acquires them all and releases to the peers at system scope once (exchange.cuh)
            am_last = atom_acq_rel_add(ticket, 1u) == gridDim.x - 1;
        __syncthreads();
        if (!am_last) return;
        if (threadIdx.x == 0) {
            *ticket = 0u;
            exch_signal(ex, -1, ep);
            exch_wait_all(ex, ep);
        }
        __syncthreads();
        // the gathered rows, after thread 0's acquire of every rank's flag and the barrier:
        // L2 loads (no stale L1 line)
        const float *src = exch_data(ex.peers[ex.rank], ex, ep);
        for (int64_t i = threadIdx.x; i < m_total; i += blockDim.x) y[i] = __ldcg(src + i);
        __syncthreads();  // every read of this epoch's data is done
        if (threadIdx.x == 0) exch_finish(ex, ep);
    }
}

// ---------------------------------------------------------------------------
// host-side configuration
// ---------------------------------------------------------------------------

template <int NMAT, int VEC, int WPR, int RG, bool XSMEM, int LB>
static cudaError_t run_gemv(const DeviceInfo &d, const GemvArgs &a, int blocks, cudaStream_t s) {
    auto kern = k_gemv<NMAT, VEC, WPR, RG, XSMEM, LB>;
    constexpr int threads = RG * WPR * kWarp;
    size_t smem = gemv_x_offset<NMAT, RG>() + (XSMEM ? (size_t)a.n * 4 : 0);
    cudaError_t e = ensure_smem(kern, d.device, smem);
    if (e != cudaSuccess) return e;
    int per_sm = 0;
    e = occupancy_cached(kern, d.device, threads, smem, &per_sm);
    if (e != cudaSuccess) return e;
    if (per_sm < 1) return cudaErrorInvalidConfiguration;
    const int64_t groups = (a.m + RG - 1) / RG;
    // a persistent wave; with >= 32 row groups per resident block, four waves
    // (later blocks fill the tail: +0.75 % at 65536 x 32768, profiles/r01j_sweep_blocks.txt)
    int64_t cap = (int64_t)per_sm * d.sms;
    if (groups >= 32 * cap) cap *= 4;
    int64_t g = blocks > 0 ? blocks : (groups < cap ? groups : cap);
    if (g < 1) g = 1;
    const int64_t wave = (int64_t)per_sm * d.sms;  // blocks of the first resident wave
    const int pf_blocks = (int)(g < wave ? g : wave);
    return launch_pdl(a.ex.world == 0, kern, dim3((unsigned)g), dim3(threads), smem, s, a.m, a.n, a.lda, a.A, a.B, a.x, a.y, a.alpha,
                      a.beta, a.epi, a.ex, a.row0, a.m_total, a.ticket, pf_blocks);
}

template <int NMAT, int VEC, bool XSMEM>
static cudaError_t dispatch_wpr(const DeviceInfo &d, int wpr, int rg, int lb, const GemvArgs &a, int blocks,
                                cudaStream_t s) {
    // block = RG row groups of WPR warps; 256..1024 threads
#define LIFT_GEMV_CASE(W, R)                                                         \
    if (wpr == W && rg == R) {                                                       \
        if (lb == 8) return run_gemv<NMAT, VEC, W, R, XSMEM, 8>(d, a, blocks, s);    \
        return run_gemv<NMAT, VEC, W, R, XSMEM, 4>(d, a, blocks, s);                 \
    }
    LIFT_GEMV_CASE(8, 1)
    LIFT_GEMV_CASE(8, 2)
    LIFT_GEMV_CASE(4, 2)
    LIFT_GEMV_CASE(4, 4)
    LIFT_GEMV_CASE(2, 4)
    LIFT_GEMV_CASE(2, 8)
    LIFT_GEMV_CASE(1, 8)
#undef LIFT_GEMV_CASE
    return cudaErrorInvalidValue;
}

template <int NMAT, int VEC, bool XSMEM, int LB>
static cudaError_t preload_set() {
    cudaFuncAttributes a;
    cudaError_t e = cudaSuccess;
#define LIFT_PRELOAD(W, R) \
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_gemv<NMAT, VEC, W, R, XSMEM, LB>);
    LIFT_PRELOAD(8, 1)
    LIFT_PRELOAD(8, 2)
    LIFT_PRELOAD(4, 2)
    LIFT_PRELOAD(4, 4)
    LIFT_PRELOAD(2, 4)
    LIFT_PRELOAD(2, 8)
    LIFT_PRELOAD(1, 8)
#undef LIFT_PRELOAD
    return e;
}

cudaError_t preload_gemv() {  // see preload_dot (dot.cu)
    cudaError_t e = set_spin_limit_here();
    if (e == cudaSuccess) e = preload_set<1, 4, true, 4>();
    if (e == cudaSuccess) e = preload_set<1, 4, true, 8>();
    if (e == cudaSuccess) e = preload_set<1, 4, false, 4>();
    if (e == cudaSuccess) e = preload_set<1, 4, false, 8>();
    if (e == cudaSuccess) e = preload_set<2, 4, true, 4>();
    if (e == cudaSuccess) e = preload_set<2, 4, true, 8>();
    if (e == cudaSuccess) e = preload_set<2, 4, false, 4>();
    if (e == cudaSuccess) e = preload_set<2, 4, false, 8>();
    cudaFuncAttributes a;
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_gemv<1, 1, 1, 8, false, 4>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_gemv<2, 1, 1, 8, false, 4>);
    return e;
}

cudaError_t launch_gemv(const DeviceInfo &d, const GemvArgs &a, GemvConfig cfg, cudaStream_t s) {
    const int64_t m = a.m, n = a.n;
    // with a fused all-gather every rank launches, even with no rows or columns of
    // its own: its peers wait for its flag (an empty row sums to 0)
    const bool exch = a.ex.world > 0;
    if (m == 0 && !exch) return cudaSuccess;
    if (n == 0 && !exch) {
        if (a.epi == kEpiStore) return cudaMemsetAsync(a.y, 0, (size_t)m * sizeof(float), s);
        // y = 0 + beta*y (and 0 when beta == 0): handled by the kernel with an empty row
    }
    uintptr_t orr = reinterpret_cast<uintptr_t>(a.A) | reinterpret_cast<uintptr_t>(a.x) |
                    (a.nmat == 2 ? reinterpret_cast<uintptr_t>(a.B) : 0);
    const bool vec = n > 0 && (n % 4 == 0) && (a.lda % 4 == 0) && (orr & 15) == 0;
    const size_t x_bytes = (size_t)n * 4;
    // Defaults from the B200 sweep (tools/sweep.py, profiles/r01b_sweep.txt): one row per
    // 256-thread block (8 warps x 1 slice each), 4 vector loads per lane per batch, x in
    // SMEM only while >= 4 blocks per SM still fit (a 128 KiB x that pins one block per SM
    // loses ~25 %; L1 serves it better).
    bool xsmem = vec && m > 0 && 4 * (x_bytes + 1024) <= (size_t)d.smem_per_sm;
    if (cfg.xsmem == 0) xsmem = false;
    if (cfg.xsmem == 1) {
        if (!(vec && x_bytes + 1024 <= (size_t)d.smem_optin)) return cudaErrorInvalidValue;
        xsmem = true;
    }
    int wpr = cfg.wpr, rg = cfg.rg;
    if (wpr == 0) wpr = vec ? 8 : 1;
    if (!vec) {
        wpr = 1;
        rg = 8;
    }
    if (rg == 0) rg = (256 / (wpr * kWarp)) > 0 ? 256 / (wpr * kWarp) : 1;
    int lb = cfg.lb;
    if (lb == 0) lb = 4;
    if (lb != 4 && lb != 8) return cudaErrorInvalidValue;
    if (vec) {
        if (a.nmat == 1)
            return xsmem ? dispatch_wpr<1, 4, true>(d, wpr, rg, lb, a, cfg.blocks, s)
                         : dispatch_wpr<1, 4, false>(d, wpr, rg, lb, a, cfg.blocks, s);
        return xsmem ? dispatch_wpr<2, 4, true>(d, wpr, rg, lb, a, cfg.blocks, s)
                     : dispatch_wpr<2, 4, false>(d, wpr, rg, lb, a, cfg.blocks, s);
    }
    // scalar path (n % 4 != 0, lda % 4 != 0 or misaligned): one shape
    if (wpr != 1 || rg != 8 || lb != 4) return cudaErrorInvalidValue;
    if (a.nmat == 1) return run_gemv<1, 1, 1, 8, false, 4>(d, a, cfg.blocks, s);
    return run_gemv<2, 1, 1, 8, false, 4>(d, a, cfg.blocks, s);
}

}  // namespace lift
