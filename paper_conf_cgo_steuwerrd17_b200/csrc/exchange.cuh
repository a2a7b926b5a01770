// exchange.cuh — the collective step fused into the kernels (SURVEY.md §8f
// NEXT-2): one-sided stores into every rank's symmetric exchange area over
// NVLink (peer pointers from torch symmetric memory / CUDA IPC), a release
// flag per (rank, epoch), and acquire-spins on the receiving side.
//
// Exchange area of every rank (same layout and size on all ranks):
//   [0, 512)      uint64 flag[64]   flag[r] = last epoch whose data rank r has
//                                   finished writing into THIS area
//   [1024, ...)   float data[2][cap] double-buffered by epoch parity
// A rank can be at most one epoch ahead of any peer (every call waits for all
// peers' flags of its own epoch), so parity double-buffering never lets a
// fast rank overwrite data a slow rank has not consumed yet.
#pragma once

#include <stdint.h>

namespace lift {

constexpr int kMaxWorld = 64;
constexpr size_t kExchHeader = 1024;

struct Exch {
    char *const *peers = nullptr;  // device array [world]: each rank's exchange area (this process's mapping)
    int rank = 0, world = 0;       // world == 0: no exchange (plain kernel)
    unsigned long long epoch = 0;  // >= 1, the same sequence of calls on every rank
    int64_t cap = 0;               // floats per parity buffer
};

__device__ __forceinline__ uint64_t *exch_flags(char *area) { return reinterpret_cast<uint64_t *>(area); }
__device__ __forceinline__ float *exch_data(char *area, const Exch &e) {
    return reinterpret_cast<float *>(area + kExchHeader) + (int64_t)(e.epoch & 1ull) * e.cap;
}

__device__ __forceinline__ void st_release_sys(uint64_t *p, uint64_t v) {
    asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ uint64_t ld_acquire_sys(const uint64_t *p) {
    uint64_t v;
    asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ float ld_volatile(const float *p) {
    float v;
    asm volatile("ld.volatile.global.f32 %0, [%1];" : "=f"(v) : "l"(p) : "memory");
    return v;
}

// After this rank's data stores to the peers: publish (caller did fence.sys).
__device__ __forceinline__ void exch_signal(const Exch &e, int dst /* -1: all ranks */) {
    for (int p = 0; p < e.world; ++p)
        if (dst < 0 || p == dst) st_release_sys(exch_flags(e.peers[p]) + e.rank, (uint64_t)e.epoch);
}

// Wait until every rank has published epoch e.epoch into THIS rank's area.
// Bounded: a peer that never arrives (a programming error) traps after ~1
// minute instead of hanging the GPU; host-side skew between ranks (allocation,
// pinning, GC) stays far below that.
__device__ __forceinline__ void exch_wait_all(const Exch &e) {
    const uint64_t *f = exch_flags(e.peers[e.rank]);
    const long long t0 = clock64();
    for (int r = 0; r < e.world; ++r) {
        while (ld_acquire_sys(f + r) < (uint64_t)e.epoch) {
            __nanosleep(100);
            if (clock64() - t0 > (1ll << 37)) __trap();  // ~70 s at 1.96 GHz
        }
    }
}

}  // namespace lift
