// pdl_probe.cu — does programmatic dependent launch (PDL) shorten a chain of
// back-to-back streaming kernels on B200?  (tuning aid, not part of the library)
//
// A graph of 20 read kernels over rotating buffers (64 or 256 MiB each, L2 never
// holds the next one), launched plainly or with programmatic stream
// serialisation: the dependent grid is scheduled early, waits in
// griddepcontrol.wait until the previous grid has completed and flushed (so it
// never reads anything the previous kernel may still write — the library's
// contract), and the previous grid allows it with griddepcontrol.launch_dependents.
// Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o tools/pdl_probe tools/pdl_probe.cu
#include <cstdint>
#include <cstdio>
#include <cuda_runtime.h>

__device__ __forceinline__ float4 ld4_na(const float4 *p) {
    float4 r;
    asm volatile("ld.global.nc.L1::no_allocate.v4.f32 {%0,%1,%2,%3}, [%4];"
                 : "=f"(r.x), "=f"(r.y), "=f"(r.z), "=f"(r.w)
                 : "l"(p));
    return r;
}

template <bool PDL>
__global__ void __launch_bounds__(256) k_read(int64_t n4, const float4 *x, float *out) {
    if constexpr (PDL) {
        asm volatile("griddepcontrol.launch_dependents;" ::: "memory");
        asm volatile("griddepcontrol.wait;" ::: "memory");
    }
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
    float4 acc[4];
    for (int u = 0; u < 4; ++u) acc[u] = make_float4(0, 0, 0, 0);
    for (; i + 3 * stride < n4; i += 4 * stride) {
        float4 a[4];
#pragma unroll
        for (int u = 0; u < 4; ++u) a[u] = ld4_na(x + i + u * stride);
#pragma unroll
        for (int u = 0; u < 4; ++u) {
            acc[u].x += a[u].x;
            acc[u].y += a[u].y;
            acc[u].z += a[u].z;
            acc[u].w += a[u].w;
        }
    }
    for (; i < n4; i += stride) acc[0].x += ld4_na(x + i).x;
    float s = 0;
    for (int u = 0; u < 4; ++u) s += acc[u].x + acc[u].y + acc[u].z + acc[u].w;
    if (s == 12345.f) out[0] = s;
}

__global__ void k_fill(float *p, int64_t n) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x)
        p[i] = (float)((uint32_t)i * 2654435761u >> 8) * 1e-7f;
}

int main() {
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    const int64_t total = (int64_t)2 << 30;  // 2 GiB of rotating buffers
    float *buf, *out;
    cudaMalloc(&buf, total);
    cudaMalloc(&out, 64);
    k_fill<<<4096, 256>>>(buf, total / 4);
    cudaDeviceSynchronize();
    cudaStream_t s;
    cudaStreamCreateWithFlags(&s, cudaStreamNonBlocking);
    for (int64_t bytes : {(int64_t)64 << 20, (int64_t)256 << 20}) {
        const int nbuf = (int)(total / bytes);
        for (int pdl = 0; pdl < 2; ++pdl) {
            for (int waves : {1, 2}) {
                const int grid = sms * 4 * waves;
                cudaGraph_t g;
                cudaGraphExec_t ge;
                cudaStreamBeginCapture(s, cudaStreamCaptureModeGlobal);
                const int calls = 20;
                for (int c = 0; c < calls; ++c) {
                    const float4 *x = (const float4 *)((char *)buf + (int64_t)(c % nbuf) * bytes);
                    cudaLaunchConfig_t cfg = {};
                    cfg.gridDim = dim3(grid);
                    cfg.blockDim = dim3(256);
                    cfg.stream = s;
                    cudaLaunchAttribute at[1];
                    at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
                    at[0].val.programmaticStreamSerializationAllowed = 1;
                    cfg.attrs = at;
                    cfg.numAttrs = pdl ? 1 : 0;
                    if (pdl)
                        cudaLaunchKernelEx(&cfg, k_read<true>, bytes / 16, x, out);
                    else
                        cudaLaunchKernelEx(&cfg, k_read<false>, bytes / 16, x, out);
                }
                cudaStreamEndCapture(s, &g);
                if (cudaGraphInstantiate(&ge, g, 0) != cudaSuccess) {
                    printf("instantiate failed: %s\n", cudaGetErrorString(cudaGetLastError()));
                    return 1;
                }
                cudaEvent_t a, b;
                cudaEventCreate(&a);
                cudaEventCreate(&b);
                float best = 1e30f;
                for (int it = 0; it < 6; ++it) {
                    cudaEventRecord(a, s);
                    cudaGraphLaunch(ge, s);
                    cudaEventRecord(b, s);
                    cudaEventSynchronize(b);
                    float ms;
                    cudaEventElapsedTime(&ms, a, b);
                    if (it >= 1 && ms < best) best = ms;
                }
                printf("%4lld MiB  grid %5d  %s  %8.2f us/launch  %7.1f GB/s\n", (long long)(bytes >> 20), grid,
                       pdl ? "PDL  " : "plain", best * 1e3 / calls, bytes * calls / (best * 1e-3) / 1e9);
                cudaGraphExecDestroy(ge);
                cudaGraphDestroy(g);
            }
        }
    }
    printf("status %s\n", cudaGetErrorString(cudaGetLastError()));
    return 0;
}
