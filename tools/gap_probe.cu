#include <cstdio>
#include <cuda_runtime.h>
__global__ void k_empty(float *o) { if (threadIdx.x == 1023) o[0] = 1.f; }
__global__ void k_one(const float *x, float *o) { float v = __ldcg(x + (size_t)blockIdx.x * 4096 + threadIdx.x); if (v == 12345.f) o[0] = v; }
int main() {
  float *o, *x; cudaMalloc(&o, 64); cudaMalloc(&x, (size_t)4 << 30);
  cudaStream_t s; cudaStreamCreate(&s);
  for (int grid : {148, 592, 1184, 2368}) for (int kind = 0; kind < 2; ++kind) {
    cudaGraph_t g; cudaGraphExec_t ge;
    cudaStreamBeginCapture(s, cudaStreamCaptureModeGlobal);
    for (int i = 0; i < 50; ++i) { if (kind == 0) k_empty<<<grid, 256, 0, s>>>(o); else k_one<<<grid, 256, 0, s>>>(x + (size_t)i * 4096 * 2368, o); }
    cudaStreamEndCapture(s, &g); cudaGraphInstantiate(&ge, g, 0);
    cudaGraphLaunch(ge, s); cudaStreamSynchronize(s);
    cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
    float best = 1e9;
    for (int r = 0; r < 5; ++r) { cudaEventRecord(a, s); cudaGraphLaunch(ge, s); cudaEventRecord(b, s); cudaEventSynchronize(b); float ms; cudaEventElapsedTime(&ms, a, b); if (ms < best) best = ms; }
    fflush(stdout); printf("%s grid %5d: %6.2f us per launch in a graph of 50\n", kind ? "one-load" : "empty   ", grid, best * 1e3 / 50);
  }
  printf("status %s\n", cudaGetErrorString(cudaGetLastError())); return 0;
}
