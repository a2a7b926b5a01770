// dot.cu — k_dot: dot(x, y) = reduce(+, 0, map(x, zip(x, y)))
//
// One launch does all three stages of Listing 1 (L391-401) plus the second
// kernel the paper omits (L422-426):
//   (1) zip + map + reduceSeq(multAndSumUp, 0): each thread folds a strided
//       chunk of float4 pairs into U independent float4 accumulators
//       (asVector4, L378-389; Fig. 7 l.10-14 = L957-961).  No product array
//       is ever formed (views instead of intermediates, L164-170).
//   (2) in-block tree (iterate, L394-397): warp butterfly, then one smem
//       exchange across warps (one barrier, Sec. 5.4).
//   (3) multi-stage: every block writes its partial (toGlobal, L393); the
//       LAST block to arrive (atomic ticket) sums all partials in a fixed
//       order and writes the scalar, then re-arms the ticket.
// mapWrg over chunks (Fig. 7 l.7-8 = L954-955) becomes a persistent
// grid-stride loop over a grid sized from the SM count.
#include "common.cuh"
#include "exchange.cuh"
#include "launch.h"

namespace lift {

template <int TPB, int U>
__device__ __forceinline__ float block_sum(float v, float *red) {
    constexpr int W = TPB / kWarp;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    v = warp_sum(v);
    if (lane == 0) red[warp] = v;
    __syncthreads();
    float r = 0.f;
    if (warp == 0) {
        r = lane < W ? red[lane] : 0.f;
        r = warp_sum(r);
    }
    return r;  // valid in warp 0
}

template <int TPB, int U, bool VEC>
__global__ void __launch_bounds__(TPB) k_dot(int64_t n, const float *__restrict__ x, const float *__restrict__ y,
                                             float *__restrict__ result, float *__restrict__ partials,
                                             unsigned int *__restrict__ ticket, Exch ex, int pf_blocks) {
    __shared__ float red[TPB / kWarp];
    __shared__ bool am_last;
    if constexpr (VEC && LIFT_PDL_PREFETCH) {
        // the first resident wave: this block's first U chunks of x and y into L2
        // while the previous kernel drains (common.cuh); lane u of warp 0 takes chunk u
        const int64_t n4 = n >> 2, i0 = (int64_t)blockIdx.x * TPB + (int64_t)threadIdx.x * gridDim.x * TPB;
        if ((int)blockIdx.x < pf_blocks && threadIdx.x < U && i0 < n4) {
            const uint32_t bytes = (uint32_t)((n4 - i0 < TPB ? n4 - i0 : TPB) * 16);
            bulk_prefetch_l2(x + 4 * i0, bytes);
            bulk_prefetch_l2(y + 4 * i0, bytes);
        }
    }
    pdl_wait();
    if (ex.world == 0) pdl_release();  // a fused collective lets nothing start early beside it
    const int64_t stride = (int64_t)gridDim.x * TPB;
    int64_t i = (int64_t)blockIdx.x * TPB + threadIdx.x;
    float s;
    if constexpr (VEC) {
        const int64_t n4 = n >> 2;
        const float4 *x4 = reinterpret_cast<const float4 *>(x);
        const float4 *y4 = reinterpret_cast<const float4 *>(y);
        float4 acc[U];
#pragma unroll
        for (int u = 0; u < U; ++u) acc[u] = zero4();
        // reduceSeq over this thread's chunk, U float4 pairs in flight per stream
        for (; i + (U - 1) * stride < n4; i += U * stride) {
            float4 a[U], b[U];
#pragma unroll
            for (int u = 0; u < U; ++u) {
                a[u] = ld_stream4(x4 + i + u * stride);
                b[u] = ld_stream4(y4 + i + u * stride);
            }
#pragma unroll
            for (int u = 0; u < U; ++u) fma4(acc[u], a[u], b[u]);
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
            if (i + u * stride < n4) fma4(acc[u], ld_stream4(x4 + i + u * stride), ld_stream4(y4 + i + u * stride));
        }
        float h[U];
#pragma unroll
        for (int u = 0; u < U; ++u) h[u] = hsum4(acc[u]);
        s = pair_tree<U>(h);
        // scalar tail (n % 4 elements) folded by block 0
        if (blockIdx.x == 0 && threadIdx.x < (n & 3)) {
            const int64_t e = (n4 << 2) + threadIdx.x;
            s = __fmaf_rn(ld_ro1(x + e), ld_ro1(y + e), s);
        }
    } else {
        float acc[4] = {0.f, 0.f, 0.f, 0.f};
        for (; i + 3 * stride < n; i += 4 * stride) {
            float a[4], b[4];
#pragma unroll
            for (int u = 0; u < 4; ++u) {
                a[u] = ld_stream1(x + i + u * stride);
                b[u] = ld_stream1(y + i + u * stride);
            }
#pragma unroll
            for (int u = 0; u < 4; ++u) acc[u] = __fmaf_rn(a[u], b[u], acc[u]);
        }
#pragma unroll
        for (int u = 0; u < 4; ++u)
            if (i + u * stride < n) acc[u] = __fmaf_rn(ld_stream1(x + i + u * stride), ld_stream1(y + i + u * stride), acc[u]);
        s = pair_tree<4>(acc);
    }

    float bs = block_sum<TPB, U>(s, red);
    if (threadIdx.x == 0) {
        partials[blockIdx.x] = bs;
        // release: publishes this block's partial; acquire: the last block then
        // sees every other block's (its threads read them after the barrier below).
        // One atom.acq_rel instead of __threadfence + atomicAdd (fence.sc is
        // stronger than needed; tools/fence_probe.py, profiles/r01w_fence_probe.txt)
        const unsigned int t = atom_acq_rel_add(ticket, 1u);
        am_last = (t == gridDim.x - 1);
    }
    __syncthreads();
    if (!am_last) return;
    // second stage (L422-426), fixed order: thread j folds partials j, j+TPB, ...
    // (8 predicated loads in flight, added in that order)
    float p = 0.f;
    for (int j0 = threadIdx.x; j0 < (int)gridDim.x; j0 += 8 * TPB) {
        float v[8];
#pragma unroll
        for (int u = 0; u < 8; ++u)
            if (j0 + u * TPB < (int)gridDim.x) v[u] = __ldcg(partials + j0 + u * TPB);
#pragma unroll
        for (int u = 0; u < 8; ++u)
            if (j0 + u * TPB < (int)gridDim.x) p = __fadd_rn(p, v[u]);
    }
    __syncthreads();  // red[] reuse
    float tot = block_sum<TPB, U>(p, red);
    if (threadIdx.x == 0) {
        *ticket = 0u;  // re-arm for the next launch on this workspace
        if (ex.world == 0) {
            *result = tot;
        } else {
            // fused all-reduce (NEXT-2): this rank's partial into slot `rank` of every
            // rank's exchange area, publish, wait for all ranks, then every rank sums
            // the slots in rank order: bitwise identical results on all ranks
            const uint64_t ep = exch_epoch(ex);
            for (int q = 0; q < ex.world; ++q) exch_data(ex.peers[q], ex, ep)[ex.rank] = tot;
            exch_signal(ex, -1, ep);  // st.release.sys: the slot stores above first
            exch_wait_all(ex, ep);
            const float *d = exch_data(ex.peers[ex.rank], ex, ep);
            float sum = 0.f;
            for (int r = 0; r < ex.world; ++r) sum = __fadd_rn(sum, ld_volatile(d + r));
            *result = sum;
            exch_finish(ex, ep);
        }
    }
}

// launch shape (tools/dot_shape_probe.py)
constexpr int kDotTPB = 256;
constexpr int kDotU = 4;
constexpr int kWaves = 2;
constexpr int64_t kUnitsPerThreadSmall = 2;
// below this many float4 units one resident wave beats two (profiles/r01w_dot_shape.txt:
// 2^22 elements 9.95 -> 8.5 us, 2^26 78.3 -> 77.1; at 2^30 two waves stay 0.6 % ahead)
constexpr int64_t kOneWaveUnits = int64_t(1) << 25;

cudaError_t launch_dot(const DeviceInfo &d, int64_t n, const float *x, const float *y, float *result,
                       void *workspace, cudaStream_t s, Exch ex) {
    // B200 read sweep (tools/readbw.cu, profiles/r01j_readbw.txt): 256-thread blocks with
    // U = 4 float4 pairs in flight per thread and TWO waves of blocks stream fastest
    // (7.48 TB/s vs 7.39 for 512 threads / one wave); later blocks fill the tail.
    constexpr int TPB = kDotTPB;
    constexpr int U = kDotU;
    unsigned int *ticket = static_cast<unsigned int *>(workspace);
    float *partials = reinterpret_cast<float *>(static_cast<char *>(workspace) + kDotTicketBytes);
    const bool vec = ((reinterpret_cast<uintptr_t>(x) | reinterpret_cast<uintptr_t>(y)) & 15) == 0;
    const int64_t units = vec ? (n >> 2) : n;
    // enough blocks to give every thread its units; at most kWaves resident waves
    int per_sm = 0;
    cudaError_t e = vec ? occupancy_cached(k_dot<TPB, U, true>, d.device, TPB, 0, &per_sm)
                        : occupancy_cached(k_dot<TPB, U, false>, d.device, TPB, 0, &per_sm);
    if (e != cudaSuccess) return e;
    if (per_sm < 1) per_sm = 1;
    // small n: two units per thread (both loads in flight in the unrolled tail) and
    // half the blocks of one unit per thread: fewer tickets and partials for the
    // second stage; 2^20: 5.2 us vs 6.7 (profiles/r01s_dot_small.txt)
    int64_t want = (units + TPB * kUnitsPerThreadSmall - 1) / (TPB * kUnitsPerThreadSmall);
    int64_t cap = (int64_t)d.sms * per_sm * (units < kOneWaveUnits ? 1 : kWaves);
    if (cap > kDotMaxBlocks) cap = kDotMaxBlocks;
    int blocks = (int)(want < 1 ? 1 : (want > cap ? cap : want));
    const int pf_blocks = d.sms * per_sm;  // blocks of the first resident wave
    if (vec) return launch_pdl(ex.world == 0, k_dot<TPB, U, true>, dim3(blocks), dim3(TPB), 0, s, n, x, y, result, partials, ticket, ex, pf_blocks);
    return launch_pdl(ex.world == 0, k_dot<TPB, U, false>, dim3(blocks), dim3(TPB), 0, s, n, x, y, result, partials, ticket, ex, pf_blocks);
}

// Load every kernel of this unit now (CUDA's lazy loading would otherwise load a
// kernel at its first launch, which waits for the device to go idle: a kernel
// spinning on a peer's flag, as the fused collectives do, would never let it).
cudaError_t preload_dot() {
    cudaFuncAttributes a;
    cudaError_t e = set_spin_limit_here();
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_dot<kDotTPB, kDotU, true>);
    if (e == cudaSuccess) e = cudaFuncGetAttributes(&a, k_dot<kDotTPB, kDotU, false>);
    return e;
}

}  // namespace lift
