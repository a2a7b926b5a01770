// atax.cu — ATAX y = A^T (A x)  (Table 1)
//
// Two algorithms, both with no materialised transpose (the transpose is the
// index l_id*N + wg_id of Fig. 6, L796-798 — element (row i, column j) of the
// row-major A at i*n + j):
//
// TWO-PASS (the paper's structure: two GEMV-shaped kernels, runtimes summed,
// L1006-1007):
//   1. t = A x          k_gemv (gemv.cu), t in the workspace (fp32)
//   2. k_atax_cols      column-blocked A^T t: block (cb, s) owns a column block
//                       and a row split; each thread owns one vector column and
//                       walks the rows of the split (a warp reads 512 contiguous
//                       bytes of a row: coalesced), folding A_ij * t_i into
//                       registers (reduceSeq, L320) -> partials[s][n]
//   3. k_colsum         y_j = sum_s partials[s][j] in a fixed order
//
// FUSED (single pass, reads A once): persistent blocks, one per SM, each owning
// a contiguous band of rows.  A producer warp streams rows of A into a ring of
// shared-memory stages with the bulk-copy engine (cp.async.bulk + mbarrier
// full/empty pairs, SASS UBLKCP).  512 consumer threads each own fixed vector
// columns with x for those columns in registers; per row they compute the
// partial dot, reduce it across the block (warp butterfly + one named barrier)
// to t_r = A_r . x, and fold A_rj * t_r into their y registers from the SAME
// registers — t is never written, A is read once (4*m*n bytes instead of 8).
// Per-block y partials are then summed by k_colsum in a fixed order.
#include <type_traits>

#include "common.cuh"
#include "launch.h"

namespace lift {

constexpr int kMaxSplits = 256;  // partial-row capacity of the workspace

static inline size_t align256(size_t b) { return (b + 255) / 256 * 256; }

size_t atax_twopass_ws_bytes(int64_t m, int64_t n) {
    return align256((size_t)m * 4) + align256((size_t)kMaxSplits * (size_t)n * 4);
}
size_t atax_fused_ws_bytes(int64_t, int64_t n) { return align256((size_t)kMaxSplits * (size_t)n * 4); }

// ---------------------------------------------------------------------------
// fixed-order column sum:  y[c] = sum_{s < S} P[s][c]
// block = 8 warps x 32 columns; warp w folds splits [w*S/8, (w+1)*S/8) in
// order, then the 8 warp partials are combined by a pairwise tree.
// ---------------------------------------------------------------------------
template <int VEC>
__global__ void __launch_bounds__(256) k_colsum(int S, int64_t nv, const float *__restrict__ P, float *__restrict__ y) {
    __shared__ __align__(16) float part[8][32 * VEC];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int64_t c = (int64_t)blockIdx.x * 32 + lane;
    const int s0 = (int)((int64_t)S * warp / 8), s1 = (int)((int64_t)S * (warp + 1) / 8);
    if constexpr (VEC == 4) {
        float4 acc = zero4();
        if (c < nv) {
            const float4 *P4 = reinterpret_cast<const float4 *>(P);
            int s = s0;
            for (; s + 4 <= s1; s += 4) {
                float4 v[4];
#pragma unroll
                for (int u = 0; u < 4; ++u) v[u] = __ldcg(P4 + (int64_t)(s + u) * nv + c);
#pragma unroll
                for (int u = 0; u < 4; ++u) {
                    acc.x = __fadd_rn(acc.x, v[u].x);
                    acc.y = __fadd_rn(acc.y, v[u].y);
                    acc.z = __fadd_rn(acc.z, v[u].z);
                    acc.w = __fadd_rn(acc.w, v[u].w);
                }
            }
            for (; s < s1; ++s) {
                float4 v = __ldcg(P4 + (int64_t)s * nv + c);
                acc.x = __fadd_rn(acc.x, v.x);
                acc.y = __fadd_rn(acc.y, v.y);
                acc.z = __fadd_rn(acc.z, v.z);
                acc.w = __fadd_rn(acc.w, v.w);
            }
        }
        reinterpret_cast<float4 *>(part[warp])[lane] = acc;
        __syncthreads();
        if (warp == 0 && c < nv) {
            float comp[4][8];
#pragma unroll
            for (int w = 0; w < 8; ++w) {
                float4 v = reinterpret_cast<const float4 *>(part[w])[lane];
                comp[0][w] = v.x;
                comp[1][w] = v.y;
                comp[2][w] = v.z;
                comp[3][w] = v.w;
            }
            float4 r = make_float4(pair_tree<8>(comp[0]), pair_tree<8>(comp[1]), pair_tree<8>(comp[2]),
                                   pair_tree<8>(comp[3]));
            reinterpret_cast<float4 *>(y)[c] = r;
        }
    } else {
        float acc = 0.f;
        if (c < nv) {
            int s = s0;
            for (; s + 4 <= s1; s += 4) {
                float v[4];
#pragma unroll
                for (int u = 0; u < 4; ++u) v[u] = __ldcg(P + (int64_t)(s + u) * nv + c);
#pragma unroll
                for (int u = 0; u < 4; ++u) acc = __fadd_rn(acc, v[u]);
            }
            for (; s < s1; ++s) acc = __fadd_rn(acc, __ldcg(P + (int64_t)s * nv + c));
        }
        part[warp][lane] = acc;
        __syncthreads();
        if (warp == 0 && c < nv) {
            float v[8];
#pragma unroll
            for (int w = 0; w < 8; ++w) v[w] = part[w][lane];
            y[c] = pair_tree<8>(v);
        }
    }
}

template <int VEC>
static cudaError_t run_colsum(int S, int64_t n, const float *P, float *y, cudaStream_t s) {
    const int64_t nv = n / VEC;
    const int64_t blocks = (nv + 31) / 32;
    k_colsum<VEC><<<(unsigned)blocks, 256, 0, s>>>(S, nv, P, y);
    return cudaGetLastError();
}

// ---------------------------------------------------------------------------
// two-pass, pass 2: partials[s][j] = sum_{i in split s} A_ij t_i
// ---------------------------------------------------------------------------
template <int VEC, int TPB, int UR>
__global__ void __launch_bounds__(TPB) k_atax_cols(int64_t m, int64_t n, int S, const float *__restrict__ A,
                                                   const float *__restrict__ t, float *__restrict__ P) {
    extern __shared__ float ts[];  // t for this row split (toLocal)
    using V = typename std::conditional<VEC == 4, float4, float>::type;
    const int s = blockIdx.y;
    const int64_t r0 = m * s / S, r1 = m * (s + 1) / S;
    for (int64_t r = r0 + threadIdx.x; r < r1; r += TPB) ts[r - r0] = __ldg(t + r);
    __syncthreads();
    const int64_t nv = n / VEC;
    const int64_t c = (int64_t)blockIdx.x * TPB + threadIdx.x;
    if (c >= nv) return;
    const V *A4 = reinterpret_cast<const V *>(A);
    V acc;
    if constexpr (VEC == 4) acc = zero4(); else acc = 0.f;
    int64_t r = r0;
    for (; r + UR <= r1; r += UR) {
        V a[UR];
#pragma unroll
        for (int u = 0; u < UR; ++u) {
            if constexpr (VEC == 4)
                a[u] = ld_stream4(A4 + (r + u) * nv + c);
            else
                a[u] = ld_stream1(A + (r + u) * n + c);
        }
#pragma unroll
        for (int u = 0; u < UR; ++u) {
            if constexpr (VEC == 4)
                fma4s(acc, a[u], ts[r + u - r0]);
            else
                acc = __fmaf_rn(a[u], ts[r + u - r0], acc);
        }
    }
    for (; r < r1; ++r) {
        if constexpr (VEC == 4)
            fma4s(acc, ld_stream4(A4 + r * nv + c), ts[r - r0]);
        else
            acc = __fmaf_rn(ld_stream1(A + r * n + c), ts[r - r0], acc);
    }
    reinterpret_cast<V *>(P)[(int64_t)s * nv + c] = acc;
}

cudaError_t launch_atax_twopass(const DeviceInfo &d, int64_t m, int64_t n, const float *A, const float *x, float *y,
                                void *ws, cudaStream_t s) {
    if (n == 0) return cudaSuccess;
    if (m == 0) return cudaMemsetAsync(y, 0, (size_t)n * 4, s);
    float *t = static_cast<float *>(ws);
    float *P = reinterpret_cast<float *>(static_cast<char *>(ws) + align256((size_t)m * 4));
    cudaError_t e = launch_gemv(d, 1, m, n, A, nullptr, x, t, 1.f, 0.f, GemvConfig{}, s);
    if (e != cudaSuccess) return e;
    const bool vec = (n % 4 == 0) && ((reinterpret_cast<uintptr_t>(A) | reinterpret_cast<uintptr_t>(y)) & 15) == 0;
    constexpr int TPB = 256;
    const int64_t nv = vec ? n / 4 : n;
    const int64_t cblocks = (nv + TPB - 1) / TPB;
    // about 8 resident 256-thread blocks per SM
    int64_t S = ((int64_t)d.sms * 8 + cblocks - 1) / cblocks;
    if (S > kMaxSplits) S = kMaxSplits;
    if (S > m) S = m;
    if (S < 1) S = 1;
    const size_t smem = (size_t)((m + S - 1) / S + 1) * 4;
    dim3 grid((unsigned)cblocks, (unsigned)S);
    if (vec) {
        auto k = k_atax_cols<4, TPB, 8>;
        if (smem > 48 * 1024) {
            e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
            if (e != cudaSuccess) return e;
        }
        k<<<grid, TPB, smem, s>>>(m, n, (int)S, A, t, P);
    } else {
        auto k = k_atax_cols<1, TPB, 8>;
        if (smem > 48 * 1024) {
            e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
            if (e != cudaSuccess) return e;
        }
        k<<<grid, TPB, smem, s>>>(m, n, (int)S, A, t, P);
    }
    e = cudaGetLastError();
    if (e != cudaSuccess) return e;
    return vec ? run_colsum<4>((int)S, n, P, y, s) : run_colsum<1>((int)S, n, P, y, s);
}

// ---------------------------------------------------------------------------
// fused single pass (bulk-copy-staged rows)
//
// Stage = one row of A (n*4 bytes) in a ring of NST shared-memory slots, each
// with a "full" mbarrier completed by the bulk-copy engine.  All 512 threads
// consume CR rows per step: CR partial dots in flight (ILP), ONE block barrier
// for all CR reductions, then CR rank-1 updates of the y registers.  The
// barrier also proves every thread has copied the step's rows into registers,
// so right after it thread 0 refills those CR slots with the rows NST ahead —
// no producer warp and no "empty" barriers are needed, and NST - CR .. NST
// rows are always in flight.
// ---------------------------------------------------------------------------
constexpr int kFusedWarps = 16;
constexpr int kFusedThreads = kFusedWarps * kWarp;  // 512
constexpr int kFusedSmemBudget = 200 * 1024;
constexpr int kFusedMaxStages = 16;
constexpr int64_t kFusedMinN = 256;  // below this, rows are too short to stream efficiently

struct FusedPlan {
    int qc;       // float4 columns per thread (1, 2, 4, 8)
    int cr;       // rows per step
    int nst;      // stages (rows) in the ring
    size_t hdr;   // barrier + reduction header bytes
    size_t smem;  // dynamic smem bytes
};

static bool fused_plan(int64_t n, FusedPlan *p) {
    if (n <= 0 || n % 4 != 0) return false;
    const int64_t nv = n / 4;
    int qc = 1;
    while (qc < 8 && (int64_t)qc * kFusedThreads < nv) qc *= 2;
    if ((int64_t)qc * kFusedThreads < nv) return false;
    const size_t row = (size_t)n * 4;
    const size_t hdr = (size_t)((8 * kFusedMaxStages + 2 * 4 * kFusedWarps * 4) + 127) / 128 * 128;
    int64_t nst = (int64_t)(((size_t)kFusedSmemBudget - hdr) / row);
    if (nst > kFusedMaxStages) nst = kFusedMaxStages;
    // rows per step: at most 4 (register budget a[cr][qc]), and small enough
    // that >= 2 further steps of rows are already in flight (lookahead)
    int cr = (int)(nst / 3);
    if (cr > 4) cr = 4;
    if (qc >= 8 && cr > 2) cr = 2;
    if (cr == 3) cr = 2;
    if (cr < 1) return false;
    if (nst < cr + 1) return false;
    p->qc = qc;
    p->cr = cr;
    p->nst = (int)nst;
    p->hdr = hdr;
    p->smem = hdr + (size_t)nst * row;
    return true;
}

bool atax_fused_supported(int64_t m, int64_t n, bool aligned16) {
    FusedPlan p;
    return aligned16 && m > 0 && fused_plan(n, &p);
}

bool atax_fused_preferred(int64_t m, int64_t n, bool aligned16) {
    return atax_fused_supported(m, n, aligned16) && n >= kFusedMinN;
}

template <int QC, int CR>
__global__ void __launch_bounds__(kFusedThreads, 1)
    k_atax_fused(int64_t m, int64_t n, int nst, int hdr, const float *__restrict__ A, const float *__restrict__ x,
                 float *__restrict__ P) {
    extern __shared__ __align__(128) unsigned char smem[];
    uint64_t *full = reinterpret_cast<uint64_t *>(smem);
    float *red = reinterpret_cast<float *>(smem + 8 * kFusedMaxStages);  // [2][CR][16]
    float *stage0 = reinterpret_cast<float *>(smem + hdr);

    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int tid = threadIdx.x;
    const int64_t nv = n / 4;
    const int64_t r0 = m * blockIdx.x / gridDim.x, r1 = m * (blockIdx.x + 1) / gridDim.x;
    const uint32_t row_bytes = (uint32_t)(n * 4);

    if (tid == 0) {
        for (int i = 0; i < nst; ++i) mbar_init(full + i, 1);
        fence_mbar_init();
    }
    __syncthreads();
    if (tid == 0) {  // prologue: fill the ring
        for (int i = 0; i < nst && r0 + i < r1; ++i) {
            mbar_arrive_expect_tx(full + i, row_bytes);
            bulk_g2s(stage0 + (size_t)i * n, A + (r0 + i) * n, row_bytes, full + i);
        }
    }

    float4 xr[QC], yr[QC];
    const float4 *x4 = reinterpret_cast<const float4 *>(x);
#pragma unroll
    for (int q = 0; q < QC; ++q) {
        const int64_t c = tid + (int64_t)kFusedThreads * q;
        xr[q] = c < nv ? ld_ro4(x4 + c) : zero4();
        yr[q] = zero4();
    }
    int it = 0, buf = 0;  // it = rows consumed so far
    for (int64_t r = r0; r < r1; r += CR, buf ^= 1) {
        const int rows = (int)((r1 - r) < CR ? (r1 - r) : CR);
        float4 a[CR][QC];
#pragma unroll
        for (int i = 0; i < CR; ++i) {
            if (i < rows) {
                const int st = (it + i) % nst;
                mbar_wait_parity(full + st, (uint32_t)(((it + i) / nst) & 1));
                const float4 *S4 = reinterpret_cast<const float4 *>(stage0 + (size_t)st * n);
#pragma unroll
                for (int q = 0; q < QC; ++q) {
                    const int64_t c = tid + (int64_t)kFusedThreads * q;
                    a[i][q] = c < nv ? S4[c] : zero4();
                }
            } else {
#pragma unroll
                for (int q = 0; q < QC; ++q) a[i][q] = zero4();
            }
        }
        // partial dots of this thread's columns, CR rows at once
        float *rb = red + buf * CR * kFusedWarps;
        float d[CR];
#pragma unroll
        for (int i = 0; i < CR; ++i) {
            float4 acc = zero4();
#pragma unroll
            for (int q = 0; q < QC; ++q) fma4(acc, a[i][q], xr[q]);
            d[i] = hsum4(acc);
        }
#pragma unroll
        for (int o = 16; o > 0; o >>= 1)
#pragma unroll
            for (int i = 0; i < CR; ++i) d[i] = __fadd_rn(d[i], __shfl_xor_sync(0xffffffffu, d[i], o));
        if (lane == 0) {
#pragma unroll
            for (int i = 0; i < CR; ++i) rb[i * kFusedWarps + warp] = d[i];
        }
        __syncthreads();  // reductions visible AND every thread is done reading this step's slots
        if (tid == 0) {
            for (int i = 0; i < rows; ++i) {
                const int64_t rn = r + i + nst;  // the row NST ahead reuses this slot
                if (rn < r1) {
                    const int st = (it + i) % nst;
                    mbar_arrive_expect_tx(full + st, row_bytes);
                    bulk_g2s(stage0 + (size_t)st * n, A + rn * n, row_bytes, full + st);
                }
            }
        }
#pragma unroll
        for (int i = 0; i < CR; ++i) {
            if (i < rows) {
                float v[kFusedWarps];
                const float4 *rb4 = reinterpret_cast<const float4 *>(rb + i * kFusedWarps);
#pragma unroll
                for (int w = 0; w < kFusedWarps / 4; ++w) {
                    const float4 t4 = rb4[w];
                    v[4 * w] = t4.x;
                    v[4 * w + 1] = t4.y;
                    v[4 * w + 2] = t4.z;
                    v[4 * w + 3] = t4.w;
                }
                const float t = pair_tree<kFusedWarps>(v);  // t_r = A_r . x
#pragma unroll
                for (int q = 0; q < QC; ++q) fma4s(yr[q], a[i][q], t);  // y += A_r^T t_r
            }
        }
        it += rows;
    }
    float4 *P4 = reinterpret_cast<float4 *>(P) + (int64_t)blockIdx.x * nv;
#pragma unroll
    for (int q = 0; q < QC; ++q) {
        const int64_t c = tid + (int64_t)kFusedThreads * q;
        if (c < nv) P4[c] = yr[q];
    }
}

template <int QC, int CR>
static cudaError_t run_fused(const FusedPlan &p, int64_t m, int64_t n, const float *A, const float *x, float *P,
                             int blocks, cudaStream_t s) {
    auto k = k_atax_fused<QC, CR>;
    cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)p.smem);
    if (e != cudaSuccess) return e;
    k<<<blocks, kFusedThreads, p.smem, s>>>(m, n, p.nst, (int)p.hdr, A, x, P);
    return cudaGetLastError();
}

cudaError_t launch_atax_fused(const DeviceInfo &d, int64_t m, int64_t n, const float *A, const float *x, float *y,
                              void *ws, cudaStream_t s) {
    if (n == 0) return cudaSuccess;
    if (m == 0) return cudaMemsetAsync(y, 0, (size_t)n * 4, s);
    FusedPlan p;
    if (!fused_plan(n, &p)) return cudaErrorInvalidValue;
    float *P = static_cast<float *>(ws);
    int64_t G = d.sms;
    if (G > kMaxSplits) G = kMaxSplits;
    if (G > m) G = m;
    cudaError_t e = cudaErrorInvalidValue;
#define LIFT_FUSED_CASE(QC, CR) \
    if (p.qc == QC && p.cr == CR) e = run_fused<QC, CR>(p, m, n, A, x, P, (int)G, s);
    LIFT_FUSED_CASE(1, 4)
    LIFT_FUSED_CASE(2, 4)
    LIFT_FUSED_CASE(4, 4)
    LIFT_FUSED_CASE(4, 2)
    LIFT_FUSED_CASE(8, 2)
    LIFT_FUSED_CASE(8, 1)
#undef LIFT_FUSED_CASE
    if (e != cudaSuccess) return e;
    return run_colsum<4>((int)G, n, P, y, s);
}

}  // namespace lift
