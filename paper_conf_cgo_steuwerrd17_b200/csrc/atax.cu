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
// a contiguous band of rows.  Thread 0 streams stages of CR rows (~32 KiB) of
// A into a ring of shared-memory slots with the bulk-copy engine (one
// cp.async.bulk + one "full" mbarrier per slot, SASS UBLKCP).  512 threads
// each own fixed vector columns with x for those columns in registers; per
// stage they compute the partial dots, reduce them across the block (warp
// butterfly + smem, one block barrier per software-pipelined step) to
// t_r = A_r . x, and fold A_rj * t_r into their y registers from the SAME
// registers — t is never written, A is read once (4*m*n bytes instead of 8).
// The per-block y partials are summed in a fixed order in the SAME launch: a
// grid barrier (cooperative launch, one block per SM) and then every block
// reduces a tile of columns over all partial rows.
//
// FUSED, WIDE ROWS (n > 16384, k_atax_fused_wide): the columns split over a
// thread-block cluster of 2..16 blocks; each block streams its column slice of the cluster's
// rows, the warps' slice dots are pushed into every block of the cluster by
// asynchronous remote stores (st.async + mbarrier complete_tx), and each row's
// rank-1 update is applied one row later from the ring.  Same second stage.
#include <mutex>
#include <type_traits>

#include "common.cuh"
#include "exchange.cuh"
#include "launch.h"

namespace lift {

constexpr int kMaxSplits = 256;  // partial-row capacity of the workspace

// Phase timestamps of the single-block fused kernel, compiled in only for the
// timeline probe (tools/atax_trace.py builds a separate library with
// -DLIFT_TRACE); the product library has none of it.
#ifdef LIFT_TRACE
constexpr int kTraceSlots = 16;
__device__ unsigned long long g_trace[kMaxSplits * kTraceSlots];
#define LIFT_STAMP(k)                                                                          \
    do {                                                                                       \
        if (threadIdx.x == 0) g_trace[blockIdx.x * kTraceSlots + (k)] = globaltimer_ns();      \
    } while (0)
#else
#define LIFT_STAMP(k) \
    do {              \
    } while (0)
#endif

static inline size_t align256(size_t b) { return (b + 255) / 256 * 256; }

// workspace: [0, 256) grid-barrier counters (zero before first use, left zero),
// then t (two-pass only), then the partial rows P[S][n]
constexpr size_t kWsHeader = 256;
size_t atax_twopass_ws_bytes(int64_t m, int64_t n) {
    return kWsHeader + align256((size_t)m * 4) + align256((size_t)kMaxSplits * (size_t)n * 4);
}
size_t atax_fused_ws_bytes(int64_t, int64_t n) { return kWsHeader + align256((size_t)kMaxSplits * (size_t)n * 4); }

// ---------------------------------------------------------------------------
// fixed-order column sum of one tile of 32 vector columns:
//   y[c] = sum_{s < S} P[s][c],  c in [c0, c0 + 32)
// W warps; warp w folds splits [w*S/W, (w+1)*S/W) in order (4 loads in
// flight), then the W warp partials are combined by a pairwise tree.  The
// order depends only on (S, W): deterministic.
// ---------------------------------------------------------------------------
template <int VEC, int W>
__device__ __forceinline__ void colsum_tile(int S, int64_t nv, const float *__restrict__ P, float *__restrict__ y,
                                            int64_t c0, float *part /* smem [W][32*VEC] */, float alpha = 1.f,
                                            float beta = 0.f, bool axpby = false) {
    using V = typename std::conditional<VEC == 4, float4, float>::type;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int64_t c = c0 + lane;
    const int s0 = (int)((int64_t)S * warp / W), s1 = (int)((int64_t)S * (warp + 1) / W);
    const V *PV = reinterpret_cast<const V *>(P);
    float acc[VEC];
#pragma unroll
    for (int e = 0; e < VEC; ++e) acc[e] = 0.f;
    if (c < nv) {
        // in order, 8 predicated loads in flight (a ragged chunk costs one L2
        // latency, not one per leftover row)
        for (int s = s0; s < s1; s += 8) {
            V v[8];
#pragma unroll
            for (int u = 0; u < 8; ++u)
                if (s + u < s1) v[u] = __ldcg(PV + (int64_t)(s + u) * nv + c);
#pragma unroll
            for (int u = 0; u < 8; ++u) {
                if (s + u < s1) {
                    const float *f = reinterpret_cast<const float *>(&v[u]);
#pragma unroll
                    for (int e = 0; e < VEC; ++e) acc[e] = __fadd_rn(acc[e], f[e]);
                }
            }
        }
    }
#pragma unroll
    for (int e = 0; e < VEC; ++e) part[(warp * 32 + lane) * VEC + e] = acc[e];
    __syncthreads();
    if (warp == 0 && c < nv) {
        float out[VEC];
#pragma unroll
        for (int e = 0; e < VEC; ++e) {
            float v[W];
#pragma unroll
            for (int w = 0; w < W; ++w) v[w] = part[(w * 32 + lane) * VEC + e];
            out[e] = pair_tree<W>(v);
            if (axpby)  // y = alpha*sum + beta*y, y not read when beta == 0 (BLAS)
                out[e] = beta == 0.f ? __fmul_rn(alpha, out[e])
                                     : __fadd_rn(__fmul_rn(alpha, out[e]), __fmul_rn(beta, y[c * VEC + e]));
        }
        if constexpr (VEC == 4)
            reinterpret_cast<float4 *>(y)[c] = make_float4(out[0], out[1], out[2], out[3]);
        else
            y[c] = out[0];
    }
    __syncthreads();  // part[] reuse by the next tile
}

constexpr int kColsumWarps = 16;

template <int VEC>
__global__ void __launch_bounds__(kColsumWarps * 32) k_colsum(int S, int64_t nv, const float *__restrict__ P,
                                                                float *__restrict__ y, float alpha, float beta,
                                                                bool axpby) {
    __shared__ __align__(16) float part[kColsumWarps * 32 * VEC];
    pdl_wait_and_release();
    colsum_tile<VEC, kColsumWarps>(S, nv, P, y, (int64_t)blockIdx.x * 32, part, alpha, beta, axpby);
}

template <int VEC>
static cudaError_t run_colsum(int S, int64_t n, const float *P, float *y, cudaStream_t s, float alpha = 1.f,
                              float beta = 0.f, bool axpby = false) {
    const int64_t nv = n / VEC;
    const int64_t blocks = (nv + 31) / 32;
    return launch_pdl(true, k_colsum<VEC>, dim3((unsigned)blocks), dim3(kColsumWarps * 32), 0, s, S, nv, P, y, alpha, beta,
                      axpby);
}

// ---------------------------------------------------------------------------
// two-pass, pass 2: partials[s][j] = sum_{i in split s} A_ij t_i
// ---------------------------------------------------------------------------
template <int VEC, int TPB, int UR>
__global__ void __launch_bounds__(TPB) k_atax_cols(int64_t m, int64_t n, int64_t lda, int S,
                                                   const float *__restrict__ A, const float *__restrict__ t,
                                                   float *__restrict__ P) {
    using V = typename std::conditional<VEC == 4, float4, float>::type;
    const int s = blockIdx.y;
    const int64_t r0 = m * s / S, r1 = m * (s + 1) / S;
    const int64_t nv = n / VEC;
    if constexpr (VEC == 4 && LIFT_PDL_PREFETCH) {
        // this block's first 2*UR row segments into L2 while the previous kernel
        // (pass 1, which writes t, never A) drains (common.cuh); one wave of blocks
        const int64_t cb = (int64_t)blockIdx.x * TPB;
        if (threadIdx.x < 2 * UR && r0 + threadIdx.x < r1 && cb < nv)
            bulk_prefetch_l2(A + (r0 + threadIdx.x) * lda + 4 * cb, (uint32_t)((nv - cb < TPB ? nv - cb : TPB) * 16));
    }
    pdl_wait_and_release();
    const int64_t c = (int64_t)blockIdx.x * TPB + threadIdx.x;
    if (c >= nv) return;
    const int64_t ldv = lda / VEC;  // row stride in vectors
    const V *AV = reinterpret_cast<const V *>(A);
    V acc;
    if constexpr (VEC == 4) acc = zero4(); else acc = 0.f;
    // rows r0, r0+1, ... in order (reduceSeq), UR rows per batch, the next batch's
    // loads issued before this one is consumed; a ragged last batch is predicated
    V cur[UR], nxt[UR];
    float tc[UR], tn[UR];  // t_i for the batch (same address across the block: broadcast)
    auto load = [&](int64_t rb, V(&a)[UR], float(&tt)[UR]) {
#pragma unroll
        for (int u = 0; u < UR; ++u) {
            if (rb + u < r1) {
                if constexpr (VEC == 4)
                    a[u] = ld_stream4(AV + (rb + u) * ldv + c);
                else
                    a[u] = ld_stream1(A + (rb + u) * lda + c);
                tt[u] = __ldg(t + rb + u);
            }
        }
    };
    if (r0 < r1) load(r0, cur, tc);
    for (int64_t r = r0; r < r1; r += UR) {
        if (r + UR < r1) load(r + UR, nxt, tn);
#pragma unroll
        for (int u = 0; u < UR; ++u) {
            if (r + u < r1) {
                if constexpr (VEC == 4)
                    fma4s(acc, cur[u], tc[u]);
                else
                    acc = __fmaf_rn(cur[u], tc[u], acc);
            }
        }
#pragma unroll
        for (int u = 0; u < UR; ++u) {
            cur[u] = nxt[u];
            tc[u] = tn[u];
        }
    }
    reinterpret_cast<V *>(P)[(int64_t)s * nv + c] = acc;
}

// partials[s][j] = sum_{i in split s} A_ij t_i, then y = colsum (with epilogue)
static cudaError_t column_pass(const DeviceInfo &d, int64_t m, int64_t n, int64_t lda, const float *A, const float *t,
                               float *P, float *y, float alpha, float beta, bool axpby, cudaStream_t s) {
    const bool vec = (n % 4 == 0) && (lda % 4 == 0) &&
                     ((reinterpret_cast<uintptr_t>(A) | reinterpret_cast<uintptr_t>(y)) & 15) == 0;
    constexpr int TPB = 256;
    const int64_t nv = vec ? n / 4 : n;
    const int64_t cblocks = (nv + TPB - 1) / TPB;
    // one resident wave: column blocks x row splits = SMs x blocks per SM
    int per_sm = 0;
    cudaError_t e = vec ? occupancy_cached(k_atax_cols<4, TPB, 8>, d.device, TPB, 0, &per_sm)
                        : occupancy_cached(k_atax_cols<1, TPB, 8>, d.device, TPB, 0, &per_sm);
    if (e != cudaSuccess) return e;
    if (per_sm < 1) per_sm = 1;
    int64_t S = (int64_t)d.sms * per_sm / cblocks;
    if (S > kMaxSplits) S = kMaxSplits;
    if (S > m) S = m;
    if (S < 1) S = 1;
    dim3 grid((unsigned)cblocks, (unsigned)S);
    e = vec ? launch_pdl(true, k_atax_cols<4, TPB, 8>, grid, dim3(TPB), 0, s, m, n, lda, (int)S, A, t, P)
            : launch_pdl(true, k_atax_cols<1, TPB, 8>, grid, dim3(TPB), 0, s, m, n, lda, (int)S, A, t, P);
    if (e != cudaSuccess) return e;
    return vec ? run_colsum<4>((int)S, n, P, y, s, alpha, beta, axpby)
               : run_colsum<1>((int)S, n, P, y, s, alpha, beta, axpby);
}

cudaError_t launch_atax_twopass(const DeviceInfo &d, int64_t m, int64_t n, const float *A, const float *x, float *y,
                                void *ws, cudaStream_t s) {
    if (n == 0) return cudaSuccess;
    if (m == 0) return cudaMemsetAsync(y, 0, (size_t)n * 4, s);
    float *t = reinterpret_cast<float *>(static_cast<char *>(ws) + kWsHeader);
    float *P = reinterpret_cast<float *>(static_cast<char *>(ws) + kWsHeader + align256((size_t)m * 4));
    GemvArgs g;
    g.m = m;
    g.n = n;
    g.lda = n;
    g.A = A;
    g.x = x;
    g.y = t;
    cudaError_t e = launch_gemv(d, g, GemvConfig{}, s);  // pass 1: t = A x
    if (e != cudaSuccess) return e;
    return column_pass(d, m, n, n, A, t, P, y, 1.f, 0.f, false, s);  // pass 2: y = A^T t
}

size_t gemv_t_ws_bytes(int64_t, int64_t n) { return kWsHeader + align256((size_t)kMaxSplits * (size_t)n * 4); }

cudaError_t launch_gemv_t(const DeviceInfo &d, int64_t m, int64_t n, int64_t lda, float alpha, const float *A,
                          const float *x, float beta, float *y, void *ws, cudaStream_t s) {
    if (n == 0) return cudaSuccess;
    if (m == 0) {  // y = beta * y (y not read when beta == 0)
        GemvArgs g;  // a 0-column GEMV over the n entries of y applies exactly that epilogue
        g.m = n;
        g.n = 0;
        g.lda = 0;
        g.y = y;
        g.alpha = alpha;
        g.beta = beta;
        g.epi = kEpiAxpby;
        return launch_gemv(d, g, GemvConfig{}, s);
    }
    float *P = reinterpret_cast<float *>(static_cast<char *>(ws) + kWsHeader);
    return column_pass(d, m, n, lda, A, x, P, y, alpha, beta, true, s);
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

// largest thread-block cluster of the wide-row kernel
constexpr int kFusedMaxCluster = 16;

struct FusedPlan {
    int qc;       // float4 columns per thread (1, 2, 4, 8)
    int cr;       // rows per step
    int nst;      // stages (rows) in the ring
    int cyc;      // 1: stages assigned to blocks cyclically, 0: contiguous bands
    size_t hdr;   // barrier + reduction header bytes
    size_t smem;  // dynamic smem bytes
};

// Stage = CR consecutive rows moved by ONE bulk copy; each consumer step takes
// one stage.  The B200 bulk-copy sweep (tools/readbw.cu bulk,
// profiles/r01p_readbw_bulk.txt) streams best with copies of >= 32 KiB and about
// 96-128 KiB in flight per SM (16 KiB copies: 5.2 TB/s; 32 KiB x 3: 7.2 TB/s;
// 32 KiB x 6: 6.5 TB/s), so CR rows make a ~32 KiB stage (within the register
// budget of two steps of a[CR][QC]) and the ring holds ~112 KiB.
constexpr size_t kFusedStageTarget = 32 * 1024;
constexpr size_t kFusedRingTarget = 112 * 1024;
constexpr int kFusedCyclic = 1;
constexpr int kFusedXsmemQc = 8;  // qc at which x moves from registers to shared memory

static bool fused_plan(int64_t n, FusedPlan *p, FusedTuning tune = FusedTuning{}) {
    if (n <= 0 || n % 4 != 0) return false;
    const int64_t nv = n / 4;
    int qc = 1;
    while (qc < 8 && (int64_t)qc * kFusedThreads < nv) qc *= 2;
    if ((int64_t)qc * kFusedThreads < nv) return false;
    const size_t row = (size_t)n * 4;
    const int cr_max = qc == 1 ? 4 : (qc == 2 ? 2 : 1);  // two steps of a[cr][qc] live in registers
    int cr = 1;
    while (cr < cr_max && (size_t)(2 * cr) * row <= kFusedStageTarget) cr *= 2;
    const size_t stage = (size_t)cr * row;
    const size_t hdr = (size_t)((8 * kFusedMaxStages + 2 * 4 * kFusedWarps * 4) + 127) / 128 * 128;
    int64_t nst = (int64_t)((kFusedRingTarget + stage / 2) / stage);
    if (nst < 2) nst = 2;
    if (nst > kFusedMaxStages) nst = kFusedMaxStages;
    // 8 float4 columns per thread: x lives in shared memory after the ring instead of
    // registers (x, y, and two steps of a row would need all 128 registers)
    const size_t xs_bytes = qc >= kFusedXsmemQc ? (size_t)n * 4 : 0;
    while (nst > 2 && hdr + (size_t)nst * stage + xs_bytes > (size_t)kFusedSmemBudget) --nst;
    if (tune.nst != 0) {  // explicit ring depth (lift_tuning.h): must fit as given
        if (tune.nst < 2 || tune.nst > kFusedMaxStages) return false;
        nst = tune.nst;
    }
    if (hdr + (size_t)nst * stage + xs_bytes > (size_t)kFusedSmemBudget) return false;
    if (tune.cyc < -1 || tune.cyc > 1) return false;
    p->qc = qc;
    p->cr = cr;
    p->nst = (int)nst;
    p->cyc = tune.cyc >= 0 ? tune.cyc : kFusedCyclic;
    p->hdr = hdr;
    // the drained ring is reused for the final column-sum tile partials
    const size_t ring = (size_t)nst * stage, tile = (size_t)kFusedWarps * 32 * 4 * sizeof(float);
    p->smem = hdr + (ring > tile ? ring : tile) + xs_bytes;
    return true;
}

// ---------------------------------------------------------------------------
// Wide rows (n > 16384: two rows and x no longer fit one block's ring): the
// columns are split over a thread-block cluster of C >= 2 blocks.  Block r of a
// cluster owns the column slice [r*n/C, (r+1)*n/C) of every row its cluster
// streams, with x and y of that slice in registers; a row's dot is the
// fixed-order sum of the C blocks' slice dots.
// ---------------------------------------------------------------------------
struct WidePlan {
    int clu;      // cluster size C (2, 4, 8 or 16); a thread owns kWideQc float4 columns of its slice
    int nst;      // ring stages (one row slice each)
    size_t hdr;   // mbarriers + pushed warp sums
    size_t smem;  // dynamic smem bytes
};

// The rank-1 update of a row is applied kWideLag steps after its dot; a thread
// owns kWideQc float4 columns of its block's slice (slices of 2049..4096 float4).
constexpr int kWideLag = 1;
constexpr int kWideLagBufs = 2 * kWideLag + 2;
constexpr int kWideQc = 8;
// Rows wider than this take the wide kernel; up to it the single-block kernel
// (whose x moves to shared memory above 8192) takes every row, tuned or not.
constexpr int64_t kWideMinN = 16384;

static size_t wide_sums_bytes(int c) {
    return 8 * kWideLagBufs + 4 * kFusedMaxStages + (size_t)kWideLagBufs * c * kFusedWarps * 4;
}

static bool wide_plan(int64_t n, WidePlan *p, FusedTuning tune = FusedTuning{}) {
    if (n <= kWideMinN || n % 4 != 0) return false;  // below: the single-block kernel
    if (tune.cyc == 0 || tune.cyc < -1 || tune.cyc > 1) return false;  // rows always go to clusters cyclically
    // the smallest cluster whose slices fit kWideQc float4 columns per thread: slices
    // of 2049..4096 float4 (32..64 KiB of a row) on as many SMs as possible — clusters
    // of 2 fill all 148 SMs (profiles/r01z_atax_wide_cluster_probe.txt)
    for (int c = 2; c <= kFusedMaxCluster; c *= 2) {
        if (n % (4 * c) != 0) continue;  // every slice a whole number of float4 columns
        const int64_t nvs = n / c / 4;
        if (nvs > kWideQc * (int64_t)kFusedThreads) continue;
        if (nvs <= 4 * (int64_t)kFusedThreads) return false;  // not reached for n > kWideMinN
        p->clu = c;
        const size_t stage = (size_t)(n / c) * 4;  // one row slice
        // as many stages as the shared-memory budget holds: a stage is refilled only
        // once every row of it has been used, so the ring is what keeps HBM busy
        const size_t hdr = (8 * kFusedMaxStages + wide_sums_bytes(c) + 127) / 128 * 128;
        int64_t nst = (int64_t)(((size_t)kFusedSmemBudget - hdr) / stage);
        if (nst < 2) nst = 2;
        if (nst < kWideLag + 2) return false;  // the lagged rows + one stage in flight
        if (nst > kFusedMaxStages) nst = kFusedMaxStages;
        if (tune.nst != 0) {
            if (tune.nst < 2 || tune.nst > kFusedMaxStages) return false;
            nst = tune.nst;
        }
        p->nst = (int)nst;
        p->hdr = hdr;
        const size_t ring = (size_t)nst * stage, tile = (size_t)kFusedWarps * 32 * 4 * sizeof(float);
        p->smem = p->hdr + (ring > tile ? ring : tile);
        return p->smem <= (size_t)kFusedSmemBudget;
    }
    return false;
}

bool atax_fused_supported(int64_t m, int64_t n, bool aligned16) {
    FusedPlan p;
    WidePlan w;
    return aligned16 && m > 0 && (fused_plan(n, &p) || wide_plan(n, &w));
}

// algo = auto: the single-block kernel from n = 256 up, the cluster kernel for
// every wider supported row — it beats the two-pass algorithm at every shape
// measured (profiles/r01z_atax_wide_cluster_probe.txt: 1.6-2.0x)
bool atax_fused_preferred(int64_t m, int64_t n, bool aligned16) {
    if (!atax_fused_supported(m, n, aligned16) || n < kFusedMinN) return false;
    FusedPlan p;
    if (fused_plan(n, &p)) return true;
    WidePlan w;
    return wide_plan(n, &w);
}

bool atax_fused_exchange_supported(int64_t m, int64_t n, bool aligned16) {
    FusedPlan p;
    return aligned16 && m > 0 && fused_plan(n, &p) && n >= kFusedMinN;
}

// Fixed-order column sum of the vector columns [c0, c1) over S partial rows,
// by one 512-thread block: 16 columns per pass, 32 row splits per column
// (each thread folds ~S/32 rows in order, all loads in flight), then the 32
// split sums of a column are combined by a pairwise tree.  Deterministic:
// the order depends only on S.
template <int IF /* loads in flight per thread */>
__device__ __forceinline__ void colsum_slice(int S, int64_t nv, const float *__restrict__ P, float *__restrict__ y,
                                             int64_t c0, int64_t c1, float4 *part /* smem [32][16] */,
                                             bool discard /* c0, c1 on 128-byte lines: drop them after use */) {
    constexpr int CW = 16, SPL = 32;
    const int tid = threadIdx.x;
    const int col = tid % CW, sp = tid / CW;
    const int s0 = (int)((int64_t)S * sp / SPL), s1 = (int)((int64_t)S * (sp + 1) / SPL);
    const float4 *P4 = reinterpret_cast<const float4 *>(P);
    for (int64_t cb = c0; cb < c1; cb += CW) {
        const int64_t c = cb + col;
        float4 acc = zero4();
        if (c < c1) {
            // in order, IF predicated loads in flight (S/32 is ~5 rows here: one
            // or two L2 latencies instead of five)
            for (int s = s0; s < s1; s += IF) {
                float4 v[IF];
#pragma unroll
                for (int u = 0; u < IF; ++u)
                    if (s + u < s1) v[u] = __ldcg(P4 + (int64_t)(s + u) * nv + c);
#pragma unroll
                for (int u = 0; u < IF; ++u) {
                    if (s + u < s1) {
                        acc.x = __fadd_rn(acc.x, v[u].x);
                        acc.y = __fadd_rn(acc.y, v[u].y);
                        acc.z = __fadd_rn(acc.z, v[u].z);
                        acc.w = __fadd_rn(acc.w, v[u].w);
                    }
                }
            }
        }
        part[sp * CW + col] = acc;
        __syncthreads();  // every load of this pass has been consumed
#ifdef LIFT_TRACE
        if (cb == c0) LIFT_STAMP(7);
#ifdef LIFT_TRACE_REPEAT  // the same loads once more (now certainly L2 hits): their latency alone
        if (cb == c0) {
            float4 acc2 = zero4();
            if (c < c1)
                for (int s = s0; s < s1; s += IF) {
                    float4 v[IF];
#pragma unroll
                    for (int u = 0; u < IF; ++u)
                        if (s + u < s1) v[u] = __ldcg(P4 + (int64_t)(s + u) * nv + c);
#pragma unroll
                    for (int u = 0; u < IF; ++u)
                        if (s + u < s1) acc2.x += v[u].x + v[u].y + v[u].z + v[u].w;
                }
            if (acc2.x == 12345.f) part[0] = acc2;  // keep the loads
            __syncthreads();
            LIFT_STAMP(8);
        }
#endif
#endif
        // one thread per (column, component) runs the pairwise tree over the 32 split
        // sums (4x shorter chains than one thread per float4 column: 16384x8192 -0.25 us,
        // 8192x32768 -0.35, profiles/r02_atax_colsum_tree64_ab.txt); same pairs, same bits
        if (tid < 4 * CW) {
            const int tc = tid >> 2, comp = tid & 3;
            if (cb + tc < c1) {
                const float *pf = reinterpret_cast<const float *>(part);
                float v[SPL];
#pragma unroll
                for (int k = 0; k < SPL; ++k) v[k] = pf[(k * CW + tc) * 4 + comp];
                y[4 * (cb + tc) + comp] = pair_tree<SPL>(v);
            }
        }
        // its lines (2 per row) of every partial row are dead now; discarded after the
        // output store is issued (-0.07 us at 4096^2, profiles/r02_atax_discard_order_ab.txt)
        if (discard) {
            const int64_t e = cb + CW < c1 ? cb + CW : c1;
            const int nl = (int)((e - cb + 7) / 8);
            for (int k = tid; k < S * nl; k += kFusedThreads)
                discard_l2_line(P4 + (int64_t)(k / nl) * nv + cb + 8 * (k % nl));
        }
        __syncthreads();
    }
}


// In-warp sums of CR row partials d[0..CR) (one per lane each), as CR
// butterflies xor 16, 8, 4, 2, 1 would give them, with the first log2(CR)
// levels folded: at level xor 16 (CR >= 2) the lower half-warp keeps rows
// [0, CR/2) and the upper half rows [CR/2, CR), each lane sending its partner
// the rows the partner keeps; at xor 8 (CR = 4) the same within each half.
// Every add pairs the same two partial sums as the plain butterfly (fp add is
// commutative), so the bits are those of CR separate butterflies.  Returns
// this lane's value; row i's sum is in lanes [i*32/CR, (i+1)*32/CR).
template <int CR>
__device__ __forceinline__ float row_butterfly(const float (&d)[CR], int lane) {
    float v;
    if constexpr (CR == 1) {
        v = d[0];
    } else if constexpr (CR == 2) {
        const bool hi = lane & 16;
        v = __fadd_rn(hi ? d[1] : d[0], __shfl_xor_sync(0xffffffffu, hi ? d[0] : d[1], 16));
    } else {
        static_assert(CR == 4, "CR is 1, 2 or 4");
        const bool hi = lane & 16;
        const float k0 = __fadd_rn(hi ? d[2] : d[0], __shfl_xor_sync(0xffffffffu, hi ? d[0] : d[2], 16));
        const float k1 = __fadd_rn(hi ? d[3] : d[1], __shfl_xor_sync(0xffffffffu, hi ? d[1] : d[3], 16));
        const bool h8 = lane & 8;
        v = __fadd_rn(h8 ? k1 : k0, __shfl_xor_sync(0xffffffffu, h8 ? k0 : k1, 8));
    }
#pragma unroll
    for (int o = 16 / CR; o > 0; o >>= 1) v = __fadd_rn(v, __shfl_xor_sync(0xffffffffu, v, o));
    return v;
}

// t[i] = pair_tree over the kFusedWarps = 16 warp sums pb[i*16 .. i*16+15]
// for i < CR, in every lane: each half-warp loads one row's 16 sums and runs
// the butterfly xor 1, 2, 4, 8, which adds exactly the pairs of the pairwise
// tree level by level (same bits as pair_tree<16>), then lane 0 / 16
// broadcasts.  Two rows per pass instead of 4 vector loads + 15 adds per row
// in every thread.
template <int CR>
__device__ __forceinline__ void warp_trees(const float *pb, int lane, float (&t)[CR]) {
    static_assert(kFusedWarps == 16, "one half-warp per row of warp sums");
#pragma unroll
    for (int i0 = 0; i0 < CR; i0 += 2) {
        const int row = (CR == 1) ? 0 : i0 + (lane >> 4);
        float v = pb[row * kFusedWarps + (lane & 15)];
#pragma unroll
        for (int o = 1; o < 16; o <<= 1) v = __fadd_rn(v, __shfl_xor_sync(0xffffffffu, v, o));
        t[i0] = __shfl_sync(0xffffffffu, v, 0);
        if (i0 + 1 < CR) t[i0 + 1] = __shfl_sync(0xffffffffu, v, 16);
    }
}

// The fused kernel's partial rows may be discarded from L2 after their last
// read only when every row is a whole number of 128-byte lines (no line shared
// by two rows).  Measured (profiles/r01u_atax_discard.txt): fused ATAX 8192^2
// 45.4 -> 44.3 us, 16384x8192 82.4 -> 81.4 us; the two-pass column sum and
// the transposed SGEMV gained nothing from it and do not discard.
static bool rows_are_lines(const float *P, int64_t n) {
    return n % 32 == 0 && (reinterpret_cast<uintptr_t>(P) & 127) == 0;
}

// One-shot grid barrier for a cooperative launch (all blocks co-resident).
// gbar[0] counts arrivals, gbar[1] departures; the last block to depart
// re-arms both to zero for the next launch on this workspace.
// Arrival: one red.release after the block barrier (publishes the block's
// partial row) or __threadfence + atomicAdd; tools/fence_probe.py.
constexpr bool kGridReleaseArrive = true;

__device__ __forceinline__ void grid_barrier(unsigned int *gbar) {
    __syncthreads();
    if (threadIdx.x == 0) {
        if constexpr (kGridReleaseArrive) {
            red_release_add(gbar, 1u);
        } else {
            __threadfence();  // publish this block's partial row
            atomicAdd(gbar, 1u);
        }
        // one thread per block polls the counter without back-off (a __nanosleep
        // between polls costs ~0.3 us per launch: profiles/r02_atax_sync_ab.txt);
        // bounded: blocks that are not all resident (a concurrent kernel holding
        // SMs under a plain launch) trap after the spin limit instead of hanging
        SpinDeadline dl;
        while (ld_acquire_gpu(gbar) < gridDim.x) dl.spin("grid barrier: not every block is resident");
    }
    __syncthreads();
}

__device__ __forceinline__ void grid_depart(unsigned int *gbar) {
    if (threadIdx.x == 0) {
        const unsigned int d = atomicAdd(gbar + 1, 1u) + 1u;
        if (d == gridDim.x) {  // every block has passed the barrier
            gbar[0] = 0u;
            gbar[1] = 0u;
        }
    }
}

template <int QC, int CR>
__global__ void __launch_bounds__(kFusedThreads, 1)
    k_atax_fused(int64_t m, int64_t n, int nst, int hdr, const float *__restrict__ A, const float *__restrict__ x,
                 float *__restrict__ P, float *__restrict__ y, unsigned int *__restrict__ gbar, Exch ex,
                 int dst, int cyc, bool discard_partials) {
    extern __shared__ __align__(128) unsigned char smem[];
    uint64_t *full = reinterpret_cast<uint64_t *>(smem);
    float *red = reinterpret_cast<float *>(smem + 8 * kFusedMaxStages);  // [2][CR][16]
    float *stage0 = reinterpret_cast<float *>(smem + hdr);

    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int tid = threadIdx.x;
    const int64_t nv = n / 4;
    const size_t stage_floats = (size_t)CR * n;
    // This block's stages (CR consecutive rows each, ONE bulk copy): either a
    // contiguous band of rows [r0, r1) (cyc = 0), or every G-th stage of the
    // whole matrix (cyc = 1: at any moment all blocks read one ~G*CR-row
    // window of A).  The assignment is fixed by (m, n, G): deterministic.
    const int64_t G = gridDim.x, bid = blockIdx.x;
    const int64_t r0 = cyc ? 0 : m * bid / G, r1 = cyc ? m : m * (bid + 1) / G;
    const int64_t all_stages = (m + CR - 1) / CR;
    const int64_t nstages = cyc ? (bid < all_stages ? (all_stages - bid + G - 1) / G : 0) : (r1 - r0 + CR - 1) / CR;
    auto stage_row = [&](int64_t j) -> int64_t { return cyc ? (j * G + bid) * CR : r0 + j * CR; };
    auto stage_rows = [&](int64_t j) -> int {
        if (j >= nstages) return 0;
        const int64_t a = stage_row(j);
        return (int)((r1 - a) < CR ? (r1 - a) : CR);
    };
    // A is read once: its lines go first when L2 needs room (-0.15..0.3 us per call,
    // profiles/r02_atax_evict_first_ab.txt)
    const uint64_t pol = l2_policy_evict_first();
    auto issue_stage = [&](int64_t j, int slot) {
        const uint32_t bytes = (uint32_t)((int64_t)stage_rows(j) * n * 4);
        mbar_arrive_expect_tx(full + slot, bytes);
        bulk_g2s_hint(stage0 + (size_t)slot * stage_floats, A + stage_row(j) * n, bytes, full + slot, pol);
    };

    if (tid == 0) {
        for (int i = 0; i < nst; ++i) mbar_init(full + i, 1);
        fence_mbar_init();
#if LIFT_PDL_PREFETCH
        // the ring's first stages into L2 while the previous kernel drains (common.cuh):
        // the whole ring when the block streams many stages, two when it streams few
        // (profiles/r02_pdl_prefetch_depth_ab.txt: 8192^2 42.95 us with the ring vs 43.4
        // with two, 4096^2 15.3 vs 15.1, 2048^2 10.0 vs 9.1; twice the ring is slower)
        const int pf = nstages <= 4 * nst ? 2 : nst;
        for (int i = 0; i < pf && i < nstages; ++i)
            bulk_prefetch_l2(A + stage_row(i) * n, (uint32_t)((int64_t)stage_rows(i) * n * 4));
#endif
    }
    __syncthreads();
    // no global access before the previous kernel is complete (a no-op unless launched
    // with the PDL attribute).  No launch_dependents: the next kernel launches at this
    // one's completion — triggered any earlier, even after the main loop, the 8 GiB-class
    // GEMV that follows in the bench step ran 17-20 us slower
    // (profiles/r02_atax_pdl_trigger_ab.txt)
    pdl_wait();
    LIFT_STAMP(0);
#ifdef LIFT_TRACE
    if (tid == 0) {  // which SM ran this block (slot 15: a value, not a time)
        unsigned int smid;
        asm volatile("mov.u32 %0, %%smid;" : "=r"(smid));
        g_trace[blockIdx.x * kTraceSlots + 15] = smid;
    }
#endif
    if (tid == 0)  // prologue: fill the ring
        for (int i = 0; i < nst && i < nstages; ++i) issue_stage(i, i);
    // fused (all-)reduce: this call's epoch (its parity buffer is free: the previous
    // call's exch_finish saw every destination done with it)
    const uint64_t ep = ex.world > 0 ? exch_epoch(ex) : 0ull;

    constexpr bool XS = QC >= kFusedXsmemQc;  // x in shared memory (after the ring) instead of registers
    float4 xr[XS ? 1 : QC], yr[QC];
    const float4 *x4 = reinterpret_cast<const float4 *>(x);
    float4 *xs4 = reinterpret_cast<float4 *>(stage0 + (size_t)nst * stage_floats);
    if constexpr (XS) {
        for (int64_t c = tid; c < nv; c += kFusedThreads) xs4[c] = ld_ro4(x4 + c);  // visible after the loop's barrier
    }
#pragma unroll
    for (int q = 0; q < QC; ++q) {
        const int64_t c = tid + (int64_t)kFusedThreads * q;
        if constexpr (!XS) xr[q] = c < nv ? ld_ro4(x4 + c) : zero4();
        yr[q] = zero4();
    }
    // Software-pipelined over steps (one step = one stage of CR rows): iteration
    // k loads stage k's rows and publishes their partial dots, then applies the
    // rank-1 updates of stage k-1 (whose block reductions are complete).  The
    // one block barrier per iteration sits at its top, where it also proves
    // that stage k-1's slot has been read into registers: thread 0 refills it
    // there with stage k-1+NST.
    int buf = 0;
    int prow = 0;        // rows of the previous stage (0: none)
    int slot = 0;        // ring slot of stage k (k % nst), tracked without division
    uint32_t phase = 0;  // its mbarrier phase parity ((k / nst) & 1)
    int pslot = 0;       // ring slot of stage k-1
    int k = 0;           // step (a block streams fewer than 2^31 stages)
    // rows of every stage but the last is CR: the per-step count is two int32
    // compares (the 64-bit stage arithmetic stays with the thread issuing copies)
    const int nstg = (int)nstages;
    const int last_rows = nstg > 0 ? stage_rows(nstg - 1) : 0;
    // Two register sets of CR rows: one step loads the current stage into `cur`
    // and applies the previous stage's updates from `prev`; steps alternate the
    // roles (no register copies between steps).  Returns true after the last.
    float4 ra[CR][QC], rb2[CR][QC];
    auto step = [&](float4(&cur)[CR][QC], float4(&prev)[CR][QC]) -> bool {
        const int rows = k < nstg - 1 ? CR : (k == nstg - 1 ? last_rows : 0);
        __syncthreads();  // previous stage: partials published, slot consumed
        if (tid == 0 && prow > 0 && k - 1 + nst < nstg) issue_stage(k - 1 + nst, pslot);
        float *rb = red + buf * CR * kFusedWarps;
        if (rows > 0) {
            mbar_wait_parity(full + slot, phase);
#ifdef LIFT_TRACE
            if (k == 0) LIFT_STAMP(1);
            if (k == nstg / 2) LIFT_STAMP(2);
#endif
            const float4 *S4 = reinterpret_cast<const float4 *>(stage0 + (size_t)slot * stage_floats);
#pragma unroll
            for (int i = 0; i < CR; ++i) {
#pragma unroll
                for (int q = 0; q < QC; ++q) {
                    const int64_t c = tid + (int64_t)kFusedThreads * q;
                    cur[i][q] = (i < rows && c < nv) ? S4[(int64_t)i * nv + c] : zero4();
                }
            }
            // partial dots of this thread's columns, CR rows at once
            float d[CR];
#pragma unroll
            for (int i = 0; i < CR; ++i) {
                float4 acc = zero4();
#pragma unroll
                for (int q = 0; q < QC; ++q) {
                    if constexpr (XS) {
                        const int64_t c = tid + (int64_t)kFusedThreads * q;
                        fma4(acc, cur[i][q], c < nv ? xs4[c] : zero4());
                    } else {
                        fma4(acc, cur[i][q], xr[q]);
                    }
                }
                d[i] = hsum4(acc);
            }
            // warp butterflies of the CR rows, folded so each level moves one value
            // per lane: row i's sum ends in lane i * 32 / CR (same bits as CR
            // separate butterflies, row_butterfly)
            const float dr = row_butterfly<CR>(d, lane);
            if ((lane & (32 / CR - 1)) == 0) rb[(lane / (32 / CR)) * kFusedWarps + warp] = dr;
        }
        // rank-1 updates of the previous stage: y += A_r^T t_r
        if (prow > 0) {
            const float *pb = red + (buf ^ 1) * CR * kFusedWarps;
            float t[CR];  // t_r = A_r . x: the pairwise tree over the 16 warp sums
            warp_trees<CR>(pb, lane, t);
#ifdef LIFT_EXP_GEMV_RING  // experiment (tools only): the ring as a GEMV, t_r written out
            if (tid == 0)
                for (int i = 0; i < CR; ++i)
                    if (i < prow) y[stage_row(k - 1) + i] = t[i];
#else
#pragma unroll
            for (int i = 0; i < CR; ++i) {
                if (i < prow) {
#pragma unroll
                    for (int q = 0; q < QC; ++q) fma4s(yr[q], prev[i][q], t[i]);
                }
            }
#endif
        }
        if (rows == 0) return true;
        prow = rows;
        pslot = slot;
        if (++slot == nst) {
            slot = 0;
            phase ^= 1u;
        }
        ++k;
        buf ^= 1;
        return false;
    };
    for (;;) {
        if (step(ra, rb2)) break;
        if (step(rb2, ra)) break;
    }
    LIFT_STAMP(3);
#ifdef LIFT_EXP_GEMV_RING
    return;
#endif
    float4 *P4 = reinterpret_cast<float4 *>(P) + (int64_t)blockIdx.x * nv;
#pragma unroll
    for (int q = 0; q < QC; ++q) {
        const int64_t c = tid + (int64_t)kFusedThreads * q;
        if (c < nv) P4[c] = yr[q];
    }

    // ---- second stage in the same launch: grid barrier, then every block sums
    // a slice of the columns over all G partial rows in a fixed order ----
    LIFT_STAMP(4);
    grid_barrier(gbar);
    LIFT_STAMP(5);
    // every block sums its own slice of columns (the drained ring holds the split sums);
    // when the partial rows are whole 128-byte lines the slices are too, and each block
    // discards the lines it has read (no DRAM write-back of dead partials)
    const bool lines = discard_partials;
    const int64_t unit = lines ? 8 : 1, nu = (nv + unit - 1) / unit;
    int64_t c0 = unit * (nu * blockIdx.x / gridDim.x), c1 = unit * (nu * (blockIdx.x + 1) / gridDim.x);
    if (c1 > nv) c1 = nv;
    colsum_slice<8>((int)gridDim.x, nv, P, y, c0, c1, reinterpret_cast<float4 *>(stage0), lines);
    LIFT_STAMP(6);
    if (ex.world == 0) {
        grid_depart(gbar);
        return;
    }
    // ---- fused reduce / all-reduce over ranks (NEXT-2): push this rank's slice of
    // A_r^T (A_r x) into row `rank` of the destination(s)' exchange area; the last
    // block of the rank publishes; every destination block then sums its slice over
    // the ranks in rank order (identical bits on every destination) ----
    const float4 *y4 = reinterpret_cast<const float4 *>(y);
    for (int q = 0; q < ex.world; ++q) {
        if (dst >= 0 && q != dst) continue;
        float4 *d4 = reinterpret_cast<float4 *>(exch_data(ex.peers[q], ex, ep) + (int64_t)ex.rank * n);
        for (int64_t c = c0 + threadIdx.x; c < c1; c += blockDim.x) d4[c] = y4[c];
    }
    __syncthreads();
    __shared__ int last_block;
    if (threadIdx.x == 0) {
        // gpu-scope release of this block's pushes; the last block acquires them all and
        // releases to the destination(s) at system scope once (exchange.cuh)
        const unsigned int dep = atom_acq_rel_add(gbar + 1, 1u) + 1u;
        last_block = dep == gridDim.x;
        if (last_block) {  // every block has pushed (and passed the grid barrier): re-arm, publish
            gbar[0] = 0u;
            gbar[1] = 0u;
            exch_signal(ex, dst, ep);
            // a rank that receives nothing is done with this epoch once it has published
            if (dst >= 0 && ex.rank != dst) exch_finish(ex, ep);
        }
    }
    if (dst >= 0 && ex.rank != dst) return;
    if (threadIdx.x == 0) exch_wait_all(ex, ep);
    __syncthreads();
    const float *src = exch_data(ex.peers[ex.rank], ex, ep);
    for (int64_t c = c0 + threadIdx.x; c < c1; c += blockDim.x) {
        float4 acc = zero4();
        for (int r = 0; r < ex.world; ++r) {  // rank order; L2 loads after thread 0's acquire + the barrier
            const float4 v = __ldcg(reinterpret_cast<const float4 *>(src + (int64_t)r * n) + c);
            acc.x = __fadd_rn(acc.x, v.x);
            acc.y = __fadd_rn(acc.y, v.y);
            acc.z = __fadd_rn(acc.z, v.z);
            acc.w = __fadd_rn(acc.w, v.w);
        }
        reinterpret_cast<float4 *>(y)[c] = acc;
    }
    // the last block to finish reading acks the epoch (its acquire sees every
    // other block's reads completed before their release-add)
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned int *readers = exch_readers(ex.peers[ex.rank]);
        if (atom_acq_rel_add(readers, 1u) == gridDim.x - 1) {
            *readers = 0u;
            exch_finish(ex, ep);
        }
    }
}

template <int QC, int CR>
static cudaError_t run_fused(const DeviceInfo &d, const FusedPlan &p, int64_t m, int64_t n, const float *A,
                             const float *x, float *P, float *y, unsigned int *gbar, int blocks, cudaStream_t s,
                             const Exch &ex, int dst, bool cooperative) {
    auto k = k_atax_fused<QC, CR>;
    cudaError_t e = ensure_smem(k, d.device, p.smem);
    if (e != cudaSuccess) return e;
    cudaLaunchAttribute attr[2];
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3((unsigned)blocks);
    cfg.blockDim = dim3(kFusedThreads);
    cfg.dynamicSmemBytes = p.smem;
    cfg.stream = s;
    cfg.attrs = attr;
    cfg.numAttrs = 0;
    if (cooperative) {  // the in-kernel grid barrier needs every block resident (one per SM)
        attr[0].id = cudaLaunchAttributeCooperative;
        attr[0].val.cooperative = 1;
        cfg.numAttrs = 1;
    }
    // programmatic dependent launch (common.cuh): the launch and this kernel's barrier
    // setup overlap the previous kernel's tail (profiles/r02_atax_pdl_ab.txt); the
    // kernel reads no global memory before its griddepcontrol.wait and never triggers
    // its own dependents early.  Not for the fused collectives (see launch_pdl).
    if (ex.world == 0 && pdl_enabled()) {
        attr[cfg.numAttrs].id = cudaLaunchAttributeProgrammaticStreamSerialization;
        attr[cfg.numAttrs].val.programmaticStreamSerializationAllowed = 1;
        ++cfg.numAttrs;
    }
    return cudaLaunchKernelEx(&cfg, k, m, n, p.nst, (int)p.hdr, A, x, P, y, gbar, ex, dst, p.cyc,
                              rows_are_lines(P, n));
}

// Wide-row fused ATAX (see WidePlan).  Cluster kc of K streams rows kc, kc+K,
// ...; its block r reads each row's column slice r (one bulk copy per row into
// a ring).  Step k computes the slice dot of row k, reduces it per warp and
// PUSHES the warp sums into every block of the cluster with asynchronous remote
// stores (st.async ... mbarrier::complete_tx), each completing bytes on the
// destination's "sums full" mbarrier of that buffer, armed by its owner with
// the step's expected bytes.  Then it applies the rank-1 update of row k-L
// (L = kWideLag) once every block's sums of that row are in: t = pairwise tree
// over the row's C x 16 sums in (block, warp) order, and the row's slice is
// re-read from the ring (a row stays in its slot until its update; the last of
// the 16 warps done with it refills the slot).  No cluster or block barrier in
// the loop, and a block waits for its peers L steps late, which absorbs their
// data-arrival jitter.  2L+2 sum buffers: a writer at step j has seen every
// block push row j-1-L, and no reader is further back than row j-1-2L.
// Second stage: partial y rows P[kc][slice] -> grid barrier -> fixed-order
// column sum over the K cluster rows.
template <int QC, int C>
__global__ void __launch_bounds__(kFusedThreads, 1)
    k_atax_fused_wide(int64_t m, int64_t n, int nst, int hdr, const float *__restrict__ A,
                          const float *__restrict__ x, float *__restrict__ P, float *__restrict__ y,
                          unsigned int *__restrict__ gbar, bool discard_partials) {
    constexpr int L = kWideLag, R = kWideLagBufs;
    extern __shared__ __align__(128) unsigned char smem[];
    uint64_t *full = reinterpret_cast<uint64_t *>(smem);
    uint64_t *sfull = full + kFusedMaxStages;                                  // [R]
    unsigned int *used = reinterpret_cast<unsigned int *>(sfull + R);         // [16]
    float *sums = reinterpret_cast<float *>(used + kFusedMaxStages);           // [R][C][16]
    float *stage0 = reinterpret_cast<float *>(smem + hdr);
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int tid = threadIdx.x;
    const int r = (int)cluster_ctarank();
    const int64_t K = cluster_count_x(), kc = cluster_id_x();
    const int64_t nc = n / C, nvs = nc / 4, col0 = (int64_t)r * nc;
    const int64_t nstages = kc < m ? (m - kc + K - 1) / K : 0;  // rows kc, kc+K, ...
    constexpr int SB = C * kFusedWarps;
    constexpr uint32_t kStepBytes = SB * 4;
    const uint64_t pol = l2_policy_evict_first();  // as k_atax_fused
    auto issue_stage = [&](int64_t j, int slot) {
        mbar_arrive_expect_tx(full + slot, (uint32_t)(nc * 4));
        bulk_g2s_hint(stage0 + (size_t)slot * nc, A + (j * K + kc) * n + col0, (uint32_t)(nc * 4), full + slot, pol);
    };
    if (tid == 0) {
        for (int i = 0; i < nst; ++i) mbar_init(full + i, 1);
        for (int i = 0; i < R; ++i) mbar_init(sfull + i, 1);
        for (int i = 0; i < kFusedMaxStages; ++i) used[i] = 0u;
        fence_mbar_init();
#if LIFT_PDL_PREFETCH
        // the ring's first row slices into L2 while the previous kernel drains (common.cuh)
        for (int i = 0; i < nst && i < nstages; ++i) bulk_prefetch_l2(A + (i * K + kc) * n + col0, (uint32_t)(nc * 4));
#endif
    }
    cluster_sync();  // every block's barriers initialised before anyone pushes into it
    pdl_wait();  // no global access before the previous kernel is complete (no early trigger: k_atax_fused)
    if (tid == 0)
        for (int i = 0; i < nst && i < nstages; ++i) issue_stage(i, i);

    const float4 *x4 = reinterpret_cast<const float4 *>(x + col0);
    float4 xr[QC], yr[QC];
#pragma unroll
    for (int q = 0; q < QC; ++q) {
        const int64_t c = tid + (int64_t)kFusedThreads * q;
        xr[q] = c < nvs ? ld_ro4(x4 + c) : zero4();
        yr[q] = zero4();
    }
    int slot = 0, sb = 0, lslot = 0, lsb = 0;
    uint32_t phase = 0, sphase = 0, lsphase = 0;
    for (int64_t k = 0; k < nstages + L; ++k) {
        if (k < nstages) {
            if (tid == 0) mbar_arrive_expect_tx(sfull + sb, kStepBytes);  // arm buffer k % R
            mbar_wait_parity(full + slot, phase);
            const float4 *S4 = reinterpret_cast<const float4 *>(stage0 + (size_t)slot * nc);
            float4 acc = zero4();
#pragma unroll
            for (int q = 0; q < QC; ++q) {
                const int64_t c = tid + (int64_t)kFusedThreads * q;
                fma4(acc, c < nvs ? S4[c] : zero4(), xr[q]);
            }
            const float dr = warp_sum(hsum4(acc));  // every lane holds the warp's sum
            const uint32_t la = smem_u32(sums + sb * SB + r * kFusedWarps + warp);
            const uint32_t lb = smem_u32(sfull + sb);
#pragma unroll
            for (int b = 0; b < C; b += 32)
                if (b + lane < C)
                    st_async_dsmem1(dsmem_addr_raw(la, (uint32_t)(b + lane)), dr, dsmem_addr_raw(lb, (uint32_t)(b + lane)));
            if (++slot == nst) {
                slot = 0;
                phase ^= 1u;
            }
            if (++sb == R) {
                sb = 0;
                sphase ^= 1u;
            }
        }
        if (k >= L) {  // the rank-1 update of row k - L
            mbar_wait_parity(sfull + lsb, lsphase);  // every block's sums of that row
            // t = pairwise tree over the row's C x 16 sums in (block, warp) order: each
            // lane's C*16/32 contiguous sums, then a butterfly over the warp
            constexpr int VPL = SB >= 32 ? SB / 32 : 1;  // C = 1: lanes 16..31 add zeros
            float v[VPL];
            const float *pb = sums + lsb * SB + lane * VPL;
#pragma unroll
            for (int u = 0; u < VPL; ++u) v[u] = (lane * VPL + u < SB) ? pb[u] : 0.f;
            float t = pair_tree<VPL>(v);
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) t = __fadd_rn(t, __shfl_xor_sync(0xffffffffu, t, o));
            const float4 *S4 = reinterpret_cast<const float4 *>(stage0 + (size_t)lslot * nc);
#pragma unroll
            for (int q = 0; q < QC; ++q) {
                const int64_t c = tid + (int64_t)kFusedThreads * q;
                if (c < nvs) fma4s(yr[q], S4[c], t);
            }
            // the last of the 16 warps done with the row's slot refills it
            __syncwarp();
            if (lane == 0) {
                if (atom_acq_rel_add_cta_shared(used + lslot, 1u) == kFusedWarps - 1) {
                    used[lslot] = 0u;
                    if (k - L + nst < nstages) issue_stage(k - L + nst, lslot);
                }
            }
            if (++lslot == nst) lslot = 0;
            if (++lsb == R) {
                lsb = 0;
                lsphase ^= 1u;
            }
        }
    }
    cluster_sync();  // no block leaves while a peer's pushes may still land in it
    float4 *P4 = reinterpret_cast<float4 *>(P + kc * n + col0);
#pragma unroll
    for (int q = 0; q < QC; ++q) {
        const int64_t c = tid + (int64_t)kFusedThreads * q;
        if (c < nvs) P4[c] = yr[q];
    }
    grid_barrier(gbar);
    const int64_t nv = n / 4;
    const bool lines = discard_partials;
    const int64_t unit = lines ? 8 : 1, nu = (nv + unit - 1) / unit;
    int64_t c0 = unit * (nu * blockIdx.x / gridDim.x), c1 = unit * (nu * (blockIdx.x + 1) / gridDim.x);
    if (c1 > nv) c1 = nv;
    colsum_slice<8>((int)K, nv, P, y, c0, c1, reinterpret_cast<float4 *>(stage0), lines);
    grid_depart(gbar);
}

template <int C>
static cudaError_t run_wide(const DeviceInfo &d, const WidePlan &p, int64_t m, int64_t n, const float *A,
                            const float *x, float *P, float *y, unsigned int *gbar, cudaStream_t s,
                            int *grid_out = nullptr /* only report the grid, launch nothing */) {
    auto k = k_atax_fused_wide<kWideQc, C>;
    cudaError_t e = ensure_smem(k, d.device, p.smem);
    if (e == cudaSuccess && C > 8) {
        static bool nonportable[64];  // set once per device
        const int dev = d.device >= 0 && d.device < 64 ? d.device : 0;
        if (!nonportable[dev]) {
            e = cudaFuncSetAttribute(k, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
            nonportable[dev] = e == cudaSuccess;
        }
    }
    if (e != cudaSuccess) return e;
    cudaLaunchAttribute attr[2];
    attr[0].id = cudaLaunchAttributeClusterDimension;
    attr[0].val.clusterDim.x = (unsigned)C;
    attr[0].val.clusterDim.y = 1;
    attr[0].val.clusterDim.z = 1;
    cudaLaunchConfig_t cfg = {};
    cfg.blockDim = dim3(kFusedThreads);
    cfg.dynamicSmemBytes = p.smem;
    cfg.stream = s;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    cfg.gridDim = dim3((unsigned)(C * (d.sms / C)));
    // every cluster resident at once (the grid barrier needs it): as many clusters
    // as the occupancy calculator says fit, cached per (device, shape)
    struct Entry {
        int dev, clu, qc, nst;
        size_t smem;
        int nc;
    };
    static Entry cache[16];
    static int used = 0;
    static std::mutex mu;
    int nc = -1;
    {
        std::lock_guard<std::mutex> lock(mu);
        for (int i = 0; i < used; ++i)
            if (cache[i].dev == d.device && cache[i].clu == C && cache[i].nst == p.nst &&
                cache[i].smem == p.smem)
                nc = cache[i].nc;
        if (nc < 0) {
            if (cudaOccupancyMaxActiveClusters(&nc, k, &cfg) != cudaSuccess) {
                (void)cudaGetLastError();
                nc = 0;
            }
            if (used < 16) cache[used++] = Entry{d.device, C, 4, p.nst, p.smem, nc};
        }
    }
    int64_t K = nc;
    if (K < 1) return cudaErrorInvalidConfiguration;
    if (K > kMaxSplits) K = kMaxSplits;
    if (K > m) K = m;
    cfg.gridDim = dim3((unsigned)(K * C));
    if (grid_out != nullptr) {
        *grid_out = (int)(K * C);
        return cudaSuccess;
    }
    // The grid barrier needs every cluster resident: ask for a cooperative launch
    // together with the cluster shape (the launch then fails instead of running a
    // grid that cannot be co-resident).  Where the driver refuses the combination
    // the launch is plain and the barrier's bounded spin is the backstop.
    // LIFT_WIDE_COOPERATIVE=0 launches plainly (a profiling aid: ncu cannot replay the
    // cooperative cluster launch — the kernel's waits time out under it).
    static int coop_ok[64];  // per device: 0 unknown, 1 accepted, -1 refused
    static const bool coop_env = [] {
        const char *v = getenv("LIFT_WIDE_COOPERATIVE");
        return !(v && v[0] == '0');
    }();
    cudaLaunchAttribute attr2[3] = {attr[0], {}, {}};
    attr2[1].id = cudaLaunchAttributeCooperative;
    attr2[1].val.cooperative = 1;
    int na2 = 2;
    if (pdl_enabled()) {  // as the single-block kernel (run_fused)
        attr[1].id = attr2[2].id = cudaLaunchAttributeProgrammaticStreamSerialization;
        attr[1].val.programmaticStreamSerializationAllowed = attr2[2].val.programmaticStreamSerializationAllowed = 1;
        cfg.numAttrs = 2;
        na2 = 3;
    }
    const int dev = d.device >= 0 && d.device < 64 ? d.device : 0;
    if (coop_env && coop_ok[dev] >= 0) {
        const int na1 = cfg.numAttrs;
        cfg.attrs = attr2;
        cfg.numAttrs = na2;
        cudaError_t e2 = cudaLaunchKernelEx(&cfg, k, m, n, p.nst, (int)p.hdr, A, x, P, y, gbar, rows_are_lines(P, n));
        if (e2 == cudaSuccess) {
            coop_ok[dev] = 1;
            return cudaSuccess;
        }
        if (coop_ok[dev] == 1) return e2;
        (void)cudaGetLastError();  // refused: remember, launch plainly
        coop_ok[dev] = -1;
        cfg.attrs = attr;
        cfg.numAttrs = na1;
    }
    return cudaLaunchKernelEx(&cfg, k, m, n, p.nst, (int)p.hdr, A, x, P, y, gbar, rows_are_lines(P, n));
}

// The grid (blocks, cluster size) lift_atax's single pass launches for (m, n)
// on this device: one block per SM (cooperative) for n <= 16384, else the
// cluster occupancy of the wide kernel (the GPC layout decides how many
// clusters fit).  Launches nothing.
cudaError_t atax_fused_grid(const DeviceInfo &d, int64_t m, int64_t n, int *blocks, int *cluster) {
    FusedPlan p;
    if (fused_plan(n, &p)) {
        int64_t G = d.sms;
        if (G > kMaxSplits) G = kMaxSplits;
        if (G > m) G = m;
        if (G < 1) G = 1;
        *blocks = (int)G;
        *cluster = 1;
        return cudaSuccess;
    }
    WidePlan w;
    if (!wide_plan(n, &w) || m < 1) return cudaErrorInvalidValue;
    *cluster = w.clu;
    if (w.clu == 2) return run_wide<2>(d, w, m, n, nullptr, nullptr, nullptr, nullptr, nullptr, 0, blocks);
    if (w.clu == 4) return run_wide<4>(d, w, m, n, nullptr, nullptr, nullptr, nullptr, nullptr, 0, blocks);
    if (w.clu == 8) return run_wide<8>(d, w, m, n, nullptr, nullptr, nullptr, nullptr, nullptr, 0, blocks);
    return run_wide<16>(d, w, m, n, nullptr, nullptr, nullptr, nullptr, nullptr, 0, blocks);
}

#ifdef LIFT_TRACE
extern "C" __attribute__((visibility("default"))) int lift_trace_copy(void *host, size_t bytes) {
    return (int)cudaMemcpyFromSymbol(host, g_trace, bytes < sizeof(g_trace) ? bytes : sizeof(g_trace));
}
#endif

cudaError_t preload_atax() {  // see preload_dot (dot.cu)
    cudaFuncAttributes a;
    cudaError_t e = set_spin_limit_here();
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused<1, 4>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused<1, 2>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused<1, 1>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused<2, 2>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused<2, 1>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused<4, 1>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused<8, 1>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused_wide<kWideQc, 2>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused_wide<kWideQc, 4>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused_wide<kWideQc, 8>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_atax_fused_wide<kWideQc, 16>);
    return e;
}

cudaError_t launch_atax_fused(const DeviceInfo &d, int64_t m, int64_t n, const float *A, const float *x, float *y,
                              void *ws, cudaStream_t s, Exch ex, int dst, int blocks, FusedTuning tune) {
    if (n == 0) return cudaSuccess;
    unsigned int *gbar = static_cast<unsigned int *>(ws);
    float *P = reinterpret_cast<float *>(static_cast<char *>(ws) + kWsHeader);
    // rows wider than 16384: the cluster kernel (single rank, grid from the cluster occupancy)
    WidePlan w;
    if (ex.world == 0 && blocks <= 0 && wide_plan(n, &w, tune)) {
        if (m == 0) return cudaMemsetAsync(y, 0, (size_t)n * 4, s);
        if (w.clu == 2) return run_wide<2>(d, w, m, n, A, x, P, y, gbar, s);
        if (w.clu == 4) return run_wide<4>(d, w, m, n, A, x, P, y, gbar, s);
        if (w.clu == 8) return run_wide<8>(d, w, m, n, A, x, P, y, gbar, s);
        if (w.clu == 16) return run_wide<16>(d, w, m, n, A, x, P, y, gbar, s);
        return cudaErrorInvalidValue;
    }
    FusedPlan p;
    if (!fused_plan(n, &p, tune)) return cudaErrorInvalidValue;
    if (m == 0 && ex.world == 0) return cudaMemsetAsync(y, 0, (size_t)n * 4, s);
    int64_t G = d.sms;
    if (G > kMaxSplits) G = kMaxSplits;
    if (G > m) G = m;
    if (G < 1) G = 1;  // m == 0 with an exchange: one block contributes a zero partial
    // cooperative launch guarantees the co-residency the grid barrier needs; an explicit
    // block count (tests running several ranks on one GPU) launches plainly
    const bool cooperative = blocks <= 0;
    if (blocks > 0) G = blocks < G ? blocks : G;
    cudaError_t e = cudaErrorInvalidValue;
#define LIFT_FUSED_CASE(QC, CR) \
    if (p.qc == QC && p.cr == CR) e = run_fused<QC, CR>(d, p, m, n, A, x, P, y, gbar, (int)G, s, ex, dst, cooperative);
    // fused_plan pairs: qc 1 -> cr 4 (rows <= 8 KiB), qc 2 -> cr 2, qc 4 / 8 -> cr 1
    LIFT_FUSED_CASE(1, 4)
    LIFT_FUSED_CASE(1, 2)
    LIFT_FUSED_CASE(1, 1)
    LIFT_FUSED_CASE(2, 2)
    LIFT_FUSED_CASE(2, 1)
    LIFT_FUSED_CASE(4, 1)
    LIFT_FUSED_CASE(8, 1)
#undef LIFT_FUSED_CASE
    return e;
}

}  // namespace lift
