// hog.cu — TEST HELPER (not part of the library): a kernel that occupies SMs
// (one block per SM through its shared-memory footprint) and spins until the
// host releases it, to check that the library's grid-barrier kernels fail
// cleanly — instead of hanging — when a concurrent kernel holds SMs.
// Built by tests/test_grid_safety_gpu.py with nvcc into a temporary directory.
#include <cuda_runtime.h>
#include <stdint.h>

static volatile int *g_flag = nullptr;  // host-mapped: 0 = hold, 1 = release
static int *g_started = nullptr;        // host-mapped: blocks that are running

__global__ void k_hog(volatile int *flag, int *started, unsigned long long limit_ns) {
    extern __shared__ char s[];
    if (threadIdx.x == 0) {
        s[0] = 1;
        atomicAdd_system(started, 1);
        unsigned long long t0, t;
        asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t0));
        do {
            __nanosleep(1000);
            asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
        } while (*flag == 0 && t - t0 < limit_ns);  // bounded: never outlives limit_ns
    }
    __syncthreads();
}

extern "C" int hog_start(int blocks, int smem_bytes, unsigned long long limit_ns, void *stream) {
    if (g_flag == nullptr) {
        if (cudaHostAlloc((void **)&g_flag, 64, cudaHostAllocMapped) != cudaSuccess) return 1;
        g_started = (int *)(g_flag + 4);
    }
    *g_flag = 0;
    *g_started = 0;
    if (cudaFuncSetAttribute(k_hog, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_bytes) != cudaSuccess) return 2;
    k_hog<<<blocks, 32, smem_bytes, (cudaStream_t)stream>>>(g_flag, g_started, limit_ns);
    return cudaGetLastError() == cudaSuccess ? 0 : 3;
}
extern "C" int hog_started(void) { return g_started ? *(volatile int *)g_started : -1; }
extern "C" void hog_release(void) {
    if (g_flag) *g_flag = 1;
}
