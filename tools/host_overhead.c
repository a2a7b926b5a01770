/* Host cost per C-ABI call, measured from C (no Python / ctypes in between):
 * N eager calls of each op on tiny device buffers (GPU work negligible), then
 * one stream sync; reports microseconds of host time per call.
 * build: gcc -O2 -Iinclude -I$CUDA/include tools/host_overhead.c \
 *          -Lpaper_conf_cgo_steuwerrd17_b200 -llift -L$CUDA/lib64 -lcudart -o /tmp/ho */
#include <stdio.h>
#include <time.h>

#include <cuda_runtime.h>

#include "lift.h"

static double now_us(void) {
    struct timespec t;
    clock_gettime(CLOCK_MONOTONIC, &t);
    return t.tv_sec * 1e6 + t.tv_nsec * 1e-3;
}

int main(void) {
    const int N = 20000;
    float *A, *x, *y, *r;
    void *wd, *wa;
    cudaMalloc((void **)&A, 64 * 1024 * 4);
    cudaMalloc((void **)&x, 1024 * 4);
    cudaMalloc((void **)&y, 1024 * 4);
    cudaMalloc((void **)&r, 16);
    size_t bd = lift_dot_workspace_bytes(1024), ba = lift_atax_workspace_bytes(64, 1024);
    cudaMalloc(&wd, bd);
    cudaMalloc(&wa, ba);
    cudaMemset(wd, 0, bd);
    cudaMemset(wa, 0, ba);
    cudaMemset(A, 0, 64 * 1024 * 4);
    cudaMemset(x, 0, 1024 * 4);
    cudaStream_t s;
    cudaStreamCreate(&s);
    for (int op = 0; op < 4; ++op) {
        const char *name[] = {"lift_dot", "lift_gemv", "lift_gesummv", "lift_atax"};
        /* batches of B calls (below the launch queue depth, so the host never waits
           for the GPU inside the timed loop), synchronised between batches */
        const int B = 256;
        for (int rep = 0; rep < 2; ++rep) {  /* first pass warms up */
            double host = 0;
            int st = 0;
            for (int b = 0; b < N / B; ++b) {
                cudaStreamSynchronize(s);
                double t0 = now_us();
                for (int i = 0; i < B; ++i) {
                    if (op == 0) st |= lift_dot(1024, x, x, r, wd, bd, (lift_stream_t)s);
                    if (op == 1) st |= lift_gemv(64, 1024, A, x, y, (lift_stream_t)s);
                    if (op == 2) st |= lift_gesummv(64, 1024, 1.5f, A, 1.2f, A, x, y, (lift_stream_t)s);
                    if (op == 3) st |= lift_atax(64, 1024, A, x, y, wa, ba, (lift_stream_t)s);
                }
                host += now_us() - t0;
            }
            cudaStreamSynchronize(s);
            if (rep == 1) printf("%-14s %6.2f us/call (host, from C)  status %d\n", name[op], host / (N / B * B), st);
        }
    }
    return 0;
}
