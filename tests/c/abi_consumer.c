/*
 * abi_consumer.c — a plain C11 program that uses the library only through
 * its C ABI (include/lift.h, lift_host.h, lift_tuning.h): no Python, no
 * torch.  It allocates with the CUDA runtime, calls each entry point on its
 * own stream, and checks every output against the fp64 oracle (oracle/,
 * test infrastructure) within the north_star tolerance
 * |y - y_ref| <= 1e-5 * mag + 1e-6, plus the documented status codes.
 *
 *   build: tests/test_c_abi.py (gcc -std=c11, links liblift.so, liboracle.so, libcudart)
 *   run:   ./abi_consumer            exit 0 = every check passed
 *          ./abi_consumer --no-gpu   status-code checks only (no device work)
 */
#include <math.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>

#include <cuda_runtime.h>

#include "lift.h"
#include "lift_host.h"
#include "lift_tuning.h"
#include "oracle.h"

static int failures = 0;

#define CHECK(cond, ...)                         \
    do {                                         \
        if (!(cond)) {                           \
            fprintf(stderr, "FAIL %s:%d: ", __FILE__, __LINE__); \
            fprintf(stderr, __VA_ARGS__);        \
            fputc('\n', stderr);                 \
            ++failures;                          \
        }                                        \
    } while (0)

#define CUDA_OK(call)                                                                      \
    do {                                                                                   \
        cudaError_t e_ = (call);                                                           \
        if (e_ != cudaSuccess) {                                                           \
            fprintf(stderr, "CUDA error %s at %s:%d\n", cudaGetErrorString(e_), __FILE__, __LINE__); \
            exit(2);                                                                       \
        }                                                                                  \
    } while (0)

/* inputs: a small xorshift generator of this test's own (U[-1, 1)) */
static uint32_t rng_state = 2463534242u;
static float urand(void) {
    rng_state ^= rng_state << 13;
    rng_state ^= rng_state >> 17;
    rng_state ^= rng_state << 5;
    return (float)((double)(rng_state >> 8) * (1.0 / 8388608.0) - 1.0);
}
static float *host_rand(int64_t count) {
    float *p = (float *)malloc((size_t)(count > 0 ? count : 1) * sizeof(float));
    for (int64_t i = 0; i < count; ++i) p[i] = urand();
    return p;
}
static float *dev_copy(const float *h, int64_t count) {
    float *d = NULL;
    CUDA_OK(cudaMalloc((void **)&d, (size_t)(count > 0 ? count : 1) * sizeof(float)));
    if (count > 0) CUDA_OK(cudaMemcpy(d, h, (size_t)count * sizeof(float), cudaMemcpyHostToDevice));
    return d;
}
static float *dev_zeros(size_t bytes) {
    float *d = NULL;
    CUDA_OK(cudaMalloc((void **)&d, bytes > 0 ? bytes : 16));
    CUDA_OK(cudaMemset(d, 0, bytes > 0 ? bytes : 16));
    return d;
}

/* elementwise north_star tolerance; returns the worst margin (<= 1 passes) */
static double margin(const float *got, const double *ref, const double *mag, int64_t count) {
    double worst = 0.0;
    for (int64_t i = 0; i < count; ++i) {
        const double err = fabs((double)got[i] - ref[i]);
        const double m = err / (1e-5 * mag[i] + 1e-6);
        if (!(m <= worst)) worst = m; /* NaN propagates as a failure */
    }
    return worst;
}

static void fetch(float *h, const float *d, int64_t count, cudaStream_t s) {
    CUDA_OK(cudaStreamSynchronize(s));
    CUDA_OK(cudaMemcpy(h, d, (size_t)count * sizeof(float), cudaMemcpyDeviceToHost));
}

static void status_codes(void) {
    /* validation happens on the host before anything touches CUDA */
    float *fake = (float *)(uintptr_t)(1u << 20); /* never dereferenced on error paths */
    char *ws = (char *)(uintptr_t)(64u << 20);
    const size_t wsb = lift_dot_workspace_bytes(100);
    CHECK(lift_dot(-1, fake, fake, fake, ws, wsb, NULL) == LIFT_ERR_BAD_SIZE, "dot bad size");
    CHECK(lift_dot(100, NULL, fake, fake + 4096, ws, wsb, NULL) == LIFT_ERR_NULL_PTR, "dot null x");
    CHECK(lift_dot(100, (float *)((char *)fake + 2), fake, fake + 4096, ws, wsb, NULL) == LIFT_ERR_MISALIGNED,
          "dot misaligned");
    CHECK(lift_dot(100, fake, fake, fake + 4096, ws, wsb - 4, NULL) == LIFT_ERR_WORKSPACE, "dot small ws");
    CHECK(lift_dot(100, fake, fake, fake + 50, ws, wsb, NULL) == LIFT_ERR_ALIAS, "dot alias");
    CHECK(lift_gemv(4, 4, fake, fake + 64, fake + 2, NULL) == LIFT_ERR_ALIAS, "gemv alias");
    CHECK(lift_gesummv(4, 4, 1.f, fake, 1.f, NULL, fake + 64, fake + 128, NULL) == LIFT_ERR_NULL_PTR, "gesummv null");
    CHECK(lift_atax_algo_run(7, 4, 4, fake, fake + 64, fake + 128, ws, 1 << 20, NULL) == LIFT_ERR_BAD_SIZE,
          "atax bad algo");
    CHECK(lift_sgemv(2, 0, 4, 4, 1.f, fake, 4, fake + 64, 0.f, fake + 128, NULL, 0, NULL) == LIFT_ERR_BAD_SIZE,
          "sgemv bad layout");
    for (int s = 0; s <= 6; ++s) CHECK(lift_strerror(s) != NULL && strlen(lift_strerror(s)) > 0, "strerror %d", s);
    CHECK(lift_strerror(12345) != NULL, "strerror unknown");
    CHECK(lift_version() > 0, "version");
}

static void dot_case(int64_t n, cudaStream_t s) {
    float *hx = host_rand(n), *hy = host_rand(n);
    float *dx = dev_copy(hx, n), *dy = dev_copy(hy, n), *dr = dev_zeros(16);
    const size_t wsb = lift_dot_workspace_bytes(n);
    float *ws = dev_zeros(wsb);
    float got = 0.f;
    for (int rep = 0; rep < 3; ++rep) { /* the ticket re-arms: repeated calls agree bitwise */
        CHECK(lift_dot(n, dx, dy, dr, ws, wsb, s) == LIFT_OK, "lift_dot n=%lld", (long long)n);
        float r;
        fetch(&r, dr, 1, s);
        if (rep == 0) got = r;
        CHECK(memcmp(&r, &got, sizeof r) == 0, "dot not reproducible");
    }
    double mag = 0.0;
    const double ref = oracle_dot(n, hx, hy, &mag);
    const double m = margin(&got, &ref, &mag, 1);
    CHECK(m <= 1.0, "dot n=%lld margin %g", (long long)n, m);
    /* host entry point: same kernels, host buffers in and out */
    float hr = -1.f;
    CHECK(lift_dot_host(n, hx, hy, &hr, dx, dy, dr, ws, wsb, s) == LIFT_OK, "lift_dot_host");
    CUDA_OK(cudaStreamSynchronize(s));
    CHECK(memcmp(&hr, &got, sizeof hr) == 0, "dot_host != dot");
    printf("dot      n=%-9lld margin %.3g\n", (long long)n, m);
    cudaFree(dx), cudaFree(dy), cudaFree(dr), cudaFree(ws), free(hx), free(hy);
}

static void gemv_case(int64_t m, int64_t n, cudaStream_t s) {
    float *hA = host_rand(m * n), *hB = host_rand(m * n), *hx = host_rand(n);
    float *dA = dev_copy(hA, m * n), *dB = dev_copy(hB, m * n), *dx = dev_copy(hx, n), *dy = dev_zeros(4 * m);
    float *got = (float *)malloc(4 * (size_t)m);
    double *ref = (double *)malloc(8 * (size_t)m), *mag = (double *)malloc(8 * (size_t)m);

    CHECK(lift_gemv(m, n, dA, dx, dy, s) == LIFT_OK, "lift_gemv");
    fetch(got, dy, m, s);
    oracle_gemv(m, n, hA, hx, ref, mag, 4);
    double mg = margin(got, ref, mag, m);
    CHECK(mg <= 1.0, "gemv %lldx%lld margin %g", (long long)m, (long long)n, mg);
    /* tuned launch shapes give the same bits (canonical row order) */
    float *got2 = (float *)malloc(4 * (size_t)m);
    CHECK(lift_gemv_tuned(m, n, dA, dx, dy, 2, 4, 0, -1, 0, s) == LIFT_OK, "lift_gemv_tuned");
    fetch(got2, dy, m, s);
    CHECK(memcmp(got, got2, 4 * (size_t)m) == 0, "gemv tuned bits differ");
    printf("gemv     %lldx%lld margin %.3g\n", (long long)m, (long long)n, mg);

    const float alpha = 1.5f, beta = -0.75f;
    CHECK(lift_gesummv(m, n, alpha, dA, beta, dB, dx, dy, s) == LIFT_OK, "lift_gesummv");
    fetch(got, dy, m, s);
    oracle_gesummv(m, n, alpha, hA, beta, hB, hx, ref, mag, 4);
    mg = margin(got, ref, mag, m);
    CHECK(mg <= 1.0, "gesummv margin %g", mg);
    printf("gesummv  %lldx%lld margin %.3g\n", (long long)m, (long long)n, mg);

    cudaFree(dA), cudaFree(dB), cudaFree(dx), cudaFree(dy);
    free(hA), free(hB), free(hx), free(got), free(got2), free(ref), free(mag);
}

static void atax_case(int64_t m, int64_t n, cudaStream_t s) {
    float *hA = host_rand(m * n), *hx = host_rand(n);
    float *dA = dev_copy(hA, m * n), *dx = dev_copy(hx, n), *dy = dev_zeros(4 * n);
    const size_t wsb = lift_atax_workspace_bytes(m, n);
    float *ws = dev_zeros(wsb);
    float *got = (float *)malloc(4 * (size_t)n);
    double *ref = (double *)malloc(8 * (size_t)n), *mag = (double *)malloc(8 * (size_t)n);
    oracle_atax(m, n, hA, hx, ref, mag, 4);
    const int algos[3] = {LIFT_ATAX_AUTO, LIFT_ATAX_FUSED, LIFT_ATAX_TWOPASS};
    for (int a = 0; a < 3; ++a) {
        const int st = lift_atax_algo_run(algos[a], m, n, dA, dx, dy, ws, wsb, s);
        if (algos[a] == LIFT_ATAX_FUSED && (n % 4 != 0 || n > 16384)) {
            CHECK(st == LIFT_ERR_BAD_SIZE, "fused must refuse n=%lld", (long long)n);
            continue;
        }
        CHECK(st == LIFT_OK, "lift_atax algo %d: %s", algos[a], lift_strerror(st));
        fetch(got, dy, n, s);
        const double mg = margin(got, ref, mag, n);
        CHECK(mg <= 1.0, "atax %lldx%lld algo %d margin %g", (long long)m, (long long)n, algos[a], mg);
        printf("atax     %lldx%lld algo %d margin %.3g\n", (long long)m, (long long)n, algos[a], mg);
    }
    cudaFree(dA), cudaFree(dx), cudaFree(dy), cudaFree(ws), free(hA), free(hx), free(got), free(ref), free(mag);
}

static void sgemv_case(int layout, int trans, int64_t m, int64_t n, int64_t pad, cudaStream_t s) {
    const int64_t rows = layout == 0 ? m : n, cols = layout == 0 ? n : m, lda = cols + pad;
    const int64_t xlen = trans == 0 ? n : m, ylen = trans == 0 ? m : n;
    float *hA = host_rand(rows * lda), *hx = host_rand(xlen), *hy = host_rand(ylen);
    float *dA = dev_copy(hA, rows * lda), *dx = dev_copy(hx, xlen), *dy = dev_copy(hy, ylen);
    const size_t wsb = lift_sgemv_workspace_bytes(layout, trans, m, n);
    float *ws = wsb ? dev_zeros(wsb) : NULL;
    const float alpha = -2.0f, beta = 0.5f;
    CHECK(lift_sgemv(layout, trans, m, n, alpha, dA, lda, dx, beta, dy, ws, wsb, s) == LIFT_OK, "lift_sgemv");
    float *got = (float *)malloc(4 * (size_t)ylen);
    double *ref = (double *)malloc(8 * (size_t)ylen), *mag = (double *)malloc(8 * (size_t)ylen);
    fetch(got, dy, ylen, s);
    oracle_sgemv(layout, trans, m, n, alpha, hA, lda, hx, beta, hy, ref, mag);
    const double mg = margin(got, ref, mag, ylen);
    CHECK(mg <= 1.0, "sgemv layout %d trans %d margin %g", layout, trans, mg);
    printf("sgemv    layout %d trans %d %lldx%lld lda %lld margin %.3g\n", layout, trans, (long long)m,
           (long long)n, (long long)lda, mg);
    cudaFree(dA), cudaFree(dx), cudaFree(dy);
    if (ws) cudaFree(ws);
    free(hA), free(hx), free(hy), free(got), free(ref), free(mag);
}

int main(int argc, char **argv) {
    printf("liblift version %d.%d\n", lift_version() >> 16, lift_version() & 0xffff);
    status_codes();
    if (argc > 1 && strcmp(argv[1], "--no-gpu") == 0) {
        printf(failures ? "ABI FAILED (%d)\n" : "ABI OK (status codes)\n", failures);
        return failures ? 1 : 0;
    }
    cudaStream_t s;
    CUDA_OK(cudaStreamCreateWithFlags(&s, cudaStreamNonBlocking));
    dot_case(0, s);
    dot_case(1, s);
    dot_case(1000003, s);
    gemv_case(1000, 1001, s);
    gemv_case(333, 4096, s);
    atax_case(777, 512, s);
    atax_case(300, 1001, s);
    for (int layout = 0; layout < 2; ++layout)
        for (int trans = 0; trans < 2; ++trans) sgemv_case(layout, trans, 301, 517, 3, s);
    CUDA_OK(cudaStreamDestroy(s));
    printf(failures ? "ABI FAILED (%d)\n" : "ABI OK\n", failures);
    return failures ? 1 : 0;
}
