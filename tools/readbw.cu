// readbw.cu — standalone B200 read-bandwidth microbenchmark (tuning aid, not
// part of the library): which load flavour / occupancy streams HBM fastest?
// Each variant sums two 4 GiB fp32 arrays (x.y) and is timed with CUDA events
// (best of 5 after 2 warm-ups).  Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

__device__ __forceinline__ float4 ld4_na(const float4 *p) {
    float4 r;
    asm volatile("ld.global.nc.L1::no_allocate.v4.f32 {%0,%1,%2,%3}, [%4];"
                 : "=f"(r.x), "=f"(r.y), "=f"(r.z), "=f"(r.w) : "l"(p));
    return r;
}
__device__ __forceinline__ float4 ld4_pf(const float4 *p) {
    float4 r;
    asm volatile("ld.global.nc.L1::no_allocate.L2::256B.v4.f32 {%0,%1,%2,%3}, [%4];"
                 : "=f"(r.x), "=f"(r.y), "=f"(r.z), "=f"(r.w) : "l"(p));
    return r;
}
struct f8 { float v[8]; };
__device__ __forceinline__ f8 ld8(const float *p) {
    f8 r;
    asm volatile("ld.global.nc.L1::no_allocate.v8.f32 {%0,%1,%2,%3,%4,%5,%6,%7}, [%8];"
                 : "=f"(r.v[0]), "=f"(r.v[1]), "=f"(r.v[2]), "=f"(r.v[3]), "=f"(r.v[4]), "=f"(r.v[5]),
                   "=f"(r.v[6]), "=f"(r.v[7]) : "l"(p));
    return r;
}
__device__ __forceinline__ f8 ld8_ef(const float *p) {
    f8 r;
    asm volatile("ld.global.nc.L1::no_allocate.L2::evict_first.v8.f32 {%0,%1,%2,%3,%4,%5,%6,%7}, [%8];"
                 : "=f"(r.v[0]), "=f"(r.v[1]), "=f"(r.v[2]), "=f"(r.v[3]), "=f"(r.v[4]), "=f"(r.v[5]),
                   "=f"(r.v[6]), "=f"(r.v[7]) : "l"(p));
    return r;
}

template <int U, int MODE>
__global__ void k4(int64_t n4, const float4 *x, const float4 *y, float *out) {
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
    float4 acc[U];
    for (int u = 0; u < U; ++u) acc[u] = make_float4(0, 0, 0, 0);
    for (; i + (U - 1) * stride < n4; i += U * stride) {
        float4 a[U], b[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            a[u] = MODE == 0 ? ld4_na(x + i + u * stride) : ld4_pf(x + i + u * stride);
            b[u] = MODE == 0 ? ld4_na(y + i + u * stride) : ld4_pf(y + i + u * stride);
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
            acc[u].x = fmaf(a[u].x, b[u].x, acc[u].x);
            acc[u].y = fmaf(a[u].y, b[u].y, acc[u].y);
            acc[u].z = fmaf(a[u].z, b[u].z, acc[u].z);
            acc[u].w = fmaf(a[u].w, b[u].w, acc[u].w);
        }
    }
    float s = 0;
    for (int u = 0; u < U; ++u) s += acc[u].x + acc[u].y + acc[u].z + acc[u].w;
    if (s == 12345.f) out[0] = s;  // keep the loads alive
}

// warp-contiguous chunks: warp w streams chunks w, w + W, ... of U*512 bytes per
// array (its U loads per array are adjacent 512-byte segments: DRAM page locality)
template <int U>
__global__ void k4c(int64_t n4, const float4 *x, const float4 *y, float *out) {
    const int lane = threadIdx.x & 31;
    const int64_t nw = (int64_t)gridDim.x * blockDim.x / 32;
    float4 acc[U];
    for (int u = 0; u < U; ++u) acc[u] = make_float4(0, 0, 0, 0);
    for (int64_t c = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) / 32; (c + 1) * U * 32 <= n4; c += nw) {
        const int64_t b = c * U * 32 + lane;
        float4 a[U], bb[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            a[u] = ld4_na(x + b + u * 32);
            bb[u] = ld4_na(y + b + u * 32);
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
            acc[u].x = fmaf(a[u].x, bb[u].x, acc[u].x);
            acc[u].y = fmaf(a[u].y, bb[u].y, acc[u].y);
            acc[u].z = fmaf(a[u].z, bb[u].z, acc[u].z);
            acc[u].w = fmaf(a[u].w, bb[u].w, acc[u].w);
        }
    }
    float s = 0;
    for (int u = 0; u < U; ++u) s += acc[u].x + acc[u].y + acc[u].z + acc[u].w;
    if (s == 12345.f) out[0] = s;
}

template <int U, int MODE>
__global__ void k8(int64_t n8, const float *x, const float *y, float *out) {
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
    float acc[8] = {0, 0, 0, 0, 0, 0, 0, 0};
    for (; i + (U - 1) * stride < n8; i += U * stride) {
        f8 a[U], b[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            a[u] = MODE == 0 ? ld8(x + 8 * (i + u * stride)) : ld8_ef(x + 8 * (i + u * stride));
            b[u] = MODE == 0 ? ld8(y + 8 * (i + u * stride)) : ld8_ef(y + 8 * (i + u * stride));
        }
#pragma unroll
        for (int u = 0; u < U; ++u)
#pragma unroll
            for (int k = 0; k < 8; ++k) acc[k] = fmaf(a[u].v[k], b[u].v[k], acc[k]);
    }
    float s = 0;
    for (int k = 0; k < 8; ++k) s += acc[k];
    if (s == 12345.f) out[0] = s;
}


// ---- bulk-copy (TMA engine) streaming: one block per SM, ring of NST slots of
// `chunk` bytes, thread 0 refills a slot as soon as the block has consumed it
__device__ __forceinline__ uint32_t su32(const void *p) { return (uint32_t)__cvta_generic_to_shared(p); }
__global__ void __launch_bounds__(256, 1) k_bulk(int64_t bytes_per_block, int chunk, int nst, const char *src,
                                                 float *out) {
    extern __shared__ __align__(128) unsigned char sm[];
    uint64_t *full = (uint64_t *)sm;
    char *ring = (char *)(sm + 1024);
    const char *base = src + (int64_t)blockIdx.x * bytes_per_block;
    const int64_t nchunks = bytes_per_block / chunk;
    if (threadIdx.x == 0) {
        for (int i = 0; i < nst; ++i) asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(su32(full + i)));
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    __syncthreads();
    auto issue = [&](int64_t c) {
        const int st = (int)(c % nst);
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(su32(full + st)), "r"(chunk)
                     : "memory");
        asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                         su32(ring + (int64_t)st * chunk)),
                     "l"(base + c * chunk), "r"(chunk), "r"(su32(full + st))
                     : "memory");
    };
    if (threadIdx.x == 0)
        for (int64_t c = 0; c < nst && c < nchunks; ++c) issue(c);
    float acc = 0.f;
    for (int64_t c = 0; c < nchunks; ++c) {
        const int st = (int)(c % nst);
        const uint32_t ph = (uint32_t)((c / nst) & 1);
        asm volatile("{\n.reg .pred p;\nW_%=:\nmbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n@!p bra W_%=;\n}\n" ::"r"(
                         su32(full + st)),
                     "r"(ph)
                     : "memory");
        const float4 *r4 = (const float4 *)(ring + (int64_t)st * chunk);
        for (int i = threadIdx.x; i < chunk / 16; i += 256) {
            float4 v = r4[i];
            acc += v.x + v.y + v.z + v.w;
        }
        __syncthreads();
        if (threadIdx.x == 0 && c + nst < nchunks) issue(c + nst);
    }
    if (acc == 12345.f) out[0] = acc;
}

// ---- bulk-copy dot: x and y streamed as chunk PAIRS into a ring of NST slot
// pairs (one mbarrier per pair), `bpsm` blocks per SM; chunk j of the grid's
// sequence goes to block j % G (cyclic: the grid reads one compact window of
// each array) or block j / per_block (banded).  TPB threads fold x.y from smem.
template <int TPB>
__global__ void __launch_bounds__(TPB) k_bulkdot(int64_t nchunks_total, int chunk, int nst, int cyclic,
                                                 const char *x, const char *y, float *out) {
    extern __shared__ __align__(128) unsigned char sm[];
    uint64_t *full = (uint64_t *)sm;
    char *ring = (char *)(sm + 1024);
    const int64_t G = gridDim.x, b = blockIdx.x;
    const int64_t mine = cyclic ? (nchunks_total - b + G - 1) / G : nchunks_total / G;
    auto src_off = [&](int64_t c) -> int64_t { return (cyclic ? c * G + b : b * mine + c) * (int64_t)chunk; };
    if (threadIdx.x == 0) {
        for (int i = 0; i < nst; ++i) asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(su32(full + i)));
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    __syncthreads();
    auto issue = [&](int64_t c) {
        const int st = (int)(c % nst);
        char *dx = ring + (int64_t)st * 2 * chunk;
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(su32(full + st)), "r"(2 * chunk)
                     : "memory");
        asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                         su32(dx)), "l"(x + src_off(c)), "r"(chunk), "r"(su32(full + st)) : "memory");
        asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                         su32(dx + chunk)), "l"(y + src_off(c)), "r"(chunk), "r"(su32(full + st)) : "memory");
    };
    if (threadIdx.x == 0)
        for (int64_t c = 0; c < nst && c < mine; ++c) issue(c);
    float4 acc = make_float4(0, 0, 0, 0);
    for (int64_t c = 0; c < mine; ++c) {
        const int st = (int)(c % nst);
        const uint32_t ph = (uint32_t)((c / nst) & 1);
        asm volatile("{\n.reg .pred p;\nW_%=:\nmbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n@!p bra W_%=;\n}\n" ::"r"(
                         su32(full + st)), "r"(ph) : "memory");
        const float4 *rx = (const float4 *)(ring + (int64_t)st * 2 * chunk);
        const float4 *ry = (const float4 *)(ring + (int64_t)st * 2 * chunk + chunk);
        for (int i = threadIdx.x; i < chunk / 16; i += TPB) {
            const float4 a = rx[i], bb = ry[i];
            acc.x = fmaf(a.x, bb.x, acc.x);
            acc.y = fmaf(a.y, bb.y, acc.y);
            acc.z = fmaf(a.z, bb.z, acc.z);
            acc.w = fmaf(a.w, bb.w, acc.w);
        }
        __syncthreads();
        if (threadIdx.x == 0 && c + nst < mine) issue(c + nst);
    }
    if (acc.x + acc.y + acc.z + acc.w == 12345.f) out[0] = 1.f;
}

// fill with non-constant data (zero pages may be served compressed)
__global__ void k_fill(float *p, int64_t n, uint32_t seed) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x) {
        uint32_t h = (uint32_t)i * 2654435761u ^ seed;
        h ^= h >> 16;
        h *= 0x7feb352du;
        h ^= h >> 15;
        p[i] = (float)(h >> 8) * (1.0f / 16777216.0f) - 0.5f;
    }
}

template <typename K, typename... Args>
static void run(const char *name, K kern, int tpb, int64_t bytes, Args... args) {
    int per_sm = 0;
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kern, tpb, 0);
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    for (int mult : {1, 2}) {
        int grid = per_sm * sms * mult;
        cudaEvent_t a, b;
        cudaEventCreate(&a);
        cudaEventCreate(&b);
        float best = 1e30f;
        for (int it = 0; it < 7; ++it) {
            cudaEventRecord(a);
            kern<<<grid, tpb>>>(args...);
            cudaEventRecord(b);
            cudaEventSynchronize(b);
            float ms;
            cudaEventElapsedTime(&ms, a, b);
            if (it >= 2 && ms < best) best = ms;
        }
        printf("%-34s tpb %4d  per_sm %2d  grid x%d  %9.1f us  %7.1f GB/s\n", name, tpb, per_sm, mult, best * 1e3,
               bytes / (best * 1e-3) / 1e9);
    }
}

int main(int argc, char **argv) {
    const int64_t n = (int64_t)1 << 30;  // 4 GiB per array
    float *x, *y, *out;
    cudaMalloc(&x, n * 4);
    cudaMalloc(&y, n * 4);
    cudaMalloc(&out, 64);
    k_fill<<<4096, 256>>>(x, n, 1u);
    k_fill<<<4096, 256>>>(y, n, 2u);
    cudaDeviceSynchronize();
    const float4 *x4 = (const float4 *)x, *y4 = (const float4 *)y;
    if (argc > 1 && argv[1][0] == 'c') {
        // grid-strided (k4) vs warp-contiguous chunks (k4c), and one 8 GiB stream vs two 4 GiB streams
        for (int rep = 0; rep < 2; ++rep) {
            run("v4 na U4 strided", k4<4, 0>, 256, 8 * n, n / 4, x4, y4, out);
            run("v4 na U4 warp-chunk 2 KiB", k4c<4>, 256, 8 * n, n / 4, x4, y4, out);
            run("v4 na U8 warp-chunk 4 KiB", k4c<8>, 256, 8 * n, n / 4, x4, y4, out);
            run("v4 na U2 warp-chunk 1 KiB", k4c<2>, 256, 8 * n, n / 4, x4, y4, out);
            // one stream: both operands from x (first and second half): 4 GiB read
            run("v4 na U4 strided, x halves", k4<4, 0>, 256, 4 * n, n / 8, x4, x4 + n / 8, out);
            run("v4 na U4 same-array 1 stream", k4<4, 0>, 256, 4 * n, n / 8, x4, x4, out);
        }
        printf("status %s\n", cudaGetErrorString(cudaGetLastError()));
        return 0;
    }
    if (argc > 1 && argv[1][0] == 'd') {
        // bulk-copy dot over x, y (4 GiB each) vs the LDG dot (k4<4,0>, 256 threads, 2 waves)
        int sms = 0;
        cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
        auto timeit = [&](auto launch) {
            cudaEvent_t a, b;
            cudaEventCreate(&a);
            cudaEventCreate(&b);
            float best = 1e30f;
            for (int it = 0; it < 6; ++it) {
                cudaEventRecord(a);
                launch();
                cudaEventRecord(b);
                cudaEventSynchronize(b);
                float ms;
                cudaEventElapsedTime(&ms, a, b);
                if (it >= 1 && ms < best) best = ms;
            }
            return best;
        };
        for (int rep = 0; rep < 2; ++rep) {
            int per_sm = 0;
            cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k4<4, 0>, 256, 0);
            float t = timeit([&] { k4<4, 0><<<per_sm * sms * 2, 256>>>(n / 4, x4, y4, out); });
            printf("ldg  dot 8 GiB  v4 na U4 256 thr x2 waves                 %9.1f us  %7.1f GB/s\n", t * 1e3,
                   8.0 * n / (t * 1e-3) / 1e9);
            for (int bpsm : {1, 2})
                for (int chunk : {16384, 32768})
                    for (int nst : {2, 3, 4})
                        for (int cyc : {0, 1}) {
                            const size_t smem = 1024 + (size_t)nst * 2 * chunk;
                            if (smem * bpsm > 225 * 1024) continue;
                            cudaFuncSetAttribute(k_bulkdot<256>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
                            const int64_t nch = 4 * n / chunk;
                            const int G = sms * bpsm;
                            float tb = timeit([&] {
                                k_bulkdot<256><<<G, 256, smem>>>(nch, chunk, nst, cyc, (const char *)x, (const char *)y, out);
                            });
                            printf("bulk dot 8 GiB  %d blk/SM chunk %5d x2  ring %d  %s  %9.1f us  %7.1f GB/s\n", bpsm,
                                   chunk, nst, cyc ? "cyclic" : "banded", tb * 1e3,
                                   (double)(cyc ? nch : nch / G * G) * chunk * 2 / (tb * 1e-3) / 1e9);
                        }
        }
        printf("status %s\n", cudaGetErrorString(cudaGetLastError()));
        return 0;
    }
    if (argc > 1 && argv[1][0] == 'b') {
        // bulk-copy streaming of 256 MiB / 2 GiB: chunk size x ring depth
        int sms = 0;
        cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
        for (int64_t total : {(int64_t)256 << 20, (int64_t)2 << 30}) {
            for (int chunk : {16384, 32768, 65536}) {
                for (int ring_kb : {96, 192}) {
                    const int nst = ring_kb * 1024 / chunk;
                    if (nst < 2) continue;
                    const int64_t per = total / sms / chunk * chunk;
                    const size_t smem = 1024 + (size_t)nst * chunk;
                    cudaFuncSetAttribute(k_bulk, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
                    cudaEvent_t a, b;
                    cudaEventCreate(&a);
                    cudaEventCreate(&b);
                    float best = 1e30f;
                    for (int it = 0; it < 7; ++it) {
                        k4<4, 0><<<4 * sms, 256>>>((int64_t)1 << 28, (const float4 *)y, (const float4 *)y, out);
                        cudaEventRecord(a);
                        k_bulk<<<sms, 256, smem>>>(per, chunk, nst, (const char *)x, out);
                        cudaEventRecord(b);
                        cudaEventSynchronize(b);
                        float ms;
                        cudaEventElapsedTime(&ms, a, b);
                        if (it >= 2 && ms < best) best = ms;
                    }
                    printf("bulk %5lld MiB chunk %6d ring %3d KiB (%2d slots)  %9.2f us  %7.1f GB/s\n",
                           (long long)(total >> 20), chunk, ring_kb, nst, best * 1e3,
                           (double)per * sms / (best * 1e-3) / 1e9);
                }
            }
        }
        printf("status %s\n", cudaGetErrorString(cudaGetLastError()));
        return 0;
    }
    if (argc > 1) {
        // size sweep: the practical read ceiling of a SINGLE launch of a given size
        // (L2 flushed by reading 1 GiB of y before each timed launch)
        for (int64_t bytes : {(int64_t)8 << 20, (int64_t)64 << 20, (int64_t)256 << 20, (int64_t)512 << 20,
                              (int64_t)2 << 30, (int64_t)4 << 30}) {
            // two arrays of bytes/8 floats each, both inside x (4 GiB)
            const int64_t m = bytes / 8;  // elements per array
            int sms = 0, per_sm = 0;
            cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
            cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k4<4, 0>, 256, 0);
            for (int mult : {1, 2}) {
                int64_t want = (m / 4 + 255) / 256;
                int64_t grid = (int64_t)per_sm * sms * mult;
                if (grid > want) grid = want;
                float best = 1e30f;
                cudaEvent_t a, b;
                cudaEventCreate(&a);
                cudaEventCreate(&b);
                for (int it = 0; it < 7; ++it) {
                    k4<4, 0><<<per_sm * sms, 256>>>((int64_t)1 << 28, (const float4 *)y, (const float4 *)y, out);
                    cudaEventRecord(a);
                    k4<4, 0><<<(int)grid, 256>>>(m / 4, x4, x4 + m / 4, out);
                    cudaEventRecord(b);
                    cudaEventSynchronize(b);
                    float ms;
                    cudaEventElapsedTime(&ms, a, b);
                    if (it >= 2 && ms < best) best = ms;
                }
                printf("single launch %6lld MiB  grid %5lld (x%d)  %9.2f us  %7.1f GB/s\n", (long long)(bytes >> 20),
                       (long long)grid, mult, best * 1e3, bytes / (best * 1e-3) / 1e9);
            }
        }
        return 0;
    }
    const int64_t bytes = 8 * n;
    run("v4 na U4", k4<4, 0>, 512, bytes, n / 4, x4, y4, out);
    run("v4 na U4", k4<4, 0>, 256, bytes, n / 4, x4, y4, out);
    run("v4 na U8", k4<8, 0>, 256, bytes, n / 4, x4, y4, out);
    run("v4 na U2", k4<2, 0>, 512, bytes, n / 4, x4, y4, out);
    run("v4 L2::256B U4", k4<4, 1>, 512, bytes, n / 4, x4, y4, out);
    run("v4 L2::256B U8", k4<8, 1>, 256, bytes, n / 4, x4, y4, out);
    run("v8 na U2", k8<2, 0>, 512, bytes, n / 8, x, y, out);
    run("v8 na U4", k8<4, 0>, 256, bytes, n / 8, x, y, out);
    run("v8 na U4", k8<4, 0>, 512, bytes, n / 8, x, y, out);
    run("v8 evict_first U4", k8<4, 1>, 256, bytes, n / 8, x, y, out);
    run("v8 evict_first U2", k8<2, 1>, 512, bytes, n / 8, x, y, out);
    cudaError_t e = cudaGetLastError();
    printf("status %s\n", cudaGetErrorString(e));
    return 0;
}
