// exchange.cuh — the collective step fused into the kernels (SURVEY.md §8f
// NEXT-2): one-sided stores into every rank's symmetric exchange area over
// NVLink (peer pointers from torch symmetric memory / CUDA IPC), a release
// flag per (rank, epoch), and acquire-spins on the receiving side.
//
// Exchange area of every rank (same layout and size on all ranks, zero before
// the first call):
//   [0, 512)      uint64 flag[64]  flag[r] = last epoch whose data rank r has
//                                  finished writing into THIS area
//   [512, 1024)   uint64 ack[64]   ack[r] = last epoch rank r has finished
//                                  with (its own reads of that epoch's data
//                                  from its own area are done); every rank
//                                  writes its ack into EVERY rank's area
//   [1024, 1028)  uint32           readers' departure counter (multi-block
//                                  consumers; zero between calls)
//   [2048, ...)   float data[2][cap]  double-buffered by epoch parity
//
// The epoch lives on the device: a call's epoch is ack[rank] of the caller's
// own area + 1 (its previous call acked epoch e - 1 there as its last act), so
// the host passes no counter and a step of fused collectives can be captured
// in a CUDA graph and replayed.
//
// Buffer reuse: the data of epoch e goes to parity e & 1, last used by epoch
// e - 2.  A rank may store epoch e's data into rank q's area only once q has
// finished reading epoch e - 2, i.e. ack[q] (in the writer's OWN area, written
// there by q) >= e - 2.  The check runs at the END of the previous call:
// after acknowledging epoch e - 1, a rank's last block waits until every
// rank's ack >= e - 2, before the kernel completes — so the next call's
// kernels, which start after it, never need it.  This holds in every mode —
// all-gather, all-reduce and reduce-to-one-rank, where the senders do not
// wait for the destination and could otherwise run two calls ahead — and in
// any mix of them.  It is a local load, normally satisfied at the first read
// (in the all-modes the flags of epoch e - 1 already imply it).
//
// Memory ordering, with as few system-scope operations as possible (a
// system-scope fence costs microseconds): the blocks of a kernel publish
// their stores into the exchange areas to ONE block of their GPU with
// gpu-scope acquire-release atomics (a ticket); that last block then releases
// at system scope (st.release.sys of the flags).  Causality is transitive in
// the PTX memory model (gpu-scope synchronisation inside the GPU, system scope
// from that block to the peers), so a peer that acquires the flag
// (ld.acquire.sys) sees every block's data.  No fence.sc / fence.acq_rel.sys
// anywhere: they measured slower than the release / acquire accesses
// (tools/fused_overhead.py, profiles/r02_fused_epilogue_ab.txt).
//
// The acknowledgements guard a write-after-read hazard only (a sender must not
// overwrite data a peer has not read yet), so they are relaxed accesses, the
// way NCCL's flag protocols treat the same hazard: a rank writes its ack after
// it has consumed the values it read (they fed the sums it stored), and a
// sender's next stores come after its check observed the ack (in a later
// kernel on the same stream).
#pragma once

#include <stdint.h>

#include "common.cuh"

namespace lift {

constexpr int kMaxWorld = 64;
constexpr size_t kExchHeader = 2048;
constexpr size_t kExchAckOff = 512;
constexpr size_t kExchReadersOff = 1024;

struct Exch {
    char *const *peers = nullptr;  // device array [world]: each rank's exchange area (this process's mapping)
    int rank = 0, world = 0;       // world == 0: no exchange (plain kernel)
    int64_t cap = 0;               // floats per parity buffer
};

__device__ __forceinline__ uint64_t *exch_flags(char *area) { return reinterpret_cast<uint64_t *>(area); }
__device__ __forceinline__ uint64_t *exch_acks(char *area) { return reinterpret_cast<uint64_t *>(area + kExchAckOff); }
__device__ __forceinline__ unsigned int *exch_readers(char *area) {
    return reinterpret_cast<unsigned int *>(area + kExchReadersOff);
}
__device__ __forceinline__ float *exch_data(char *area, const Exch &e, uint64_t epoch) {
    return reinterpret_cast<float *>(area + kExchHeader) + (int64_t)(epoch & 1ull) * e.cap;
}

__device__ __forceinline__ void st_release_sys(uint64_t *p, uint64_t v) {
    asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ uint64_t ld_acquire_sys(const uint64_t *p) {
    uint64_t v;
    asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ uint64_t ld_relaxed_sys(const uint64_t *p) {
    uint64_t v;
    asm volatile("ld.relaxed.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ void st_relaxed_sys(uint64_t *p, uint64_t v) {
    asm volatile("st.relaxed.sys.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ void fence_acq_rel_sys() { asm volatile("fence.acq_rel.sys;" ::: "memory"); }
__device__ __forceinline__ float ld_volatile(const float *p) {
    float v;
    asm volatile("ld.volatile.global.f32 %0, [%1];" : "=f"(v) : "l"(p) : "memory");
    return v;
}

// This call's epoch: one more than the last epoch this rank acked into its own area.
__device__ __forceinline__ uint64_t exch_epoch(const Exch &e) {
    return ld_relaxed_sys(exch_acks(e.peers[e.rank]) + e.rank) + 1ull;
}

// After this rank's data stores to the peers (this thread's own, and every
// other block's, acquired through a gpu-scope ticket): publish, one release.
__device__ __forceinline__ void exch_signal(const Exch &e, int dst /* -1: all ranks */, uint64_t epoch) {
    for (int p = 0; p < e.world; ++p)
        if (dst < 0 || p == dst) st_release_sys(exch_flags(e.peers[p]) + e.rank, epoch);
}

// Wait until every rank has published `epoch` into THIS rank's area.  Bounded:
// a peer that never arrives (a programming error) traps instead of hanging the
// GPU; host-side skew between ranks (allocation, pinning, GC) stays far below
// the limit.
__device__ __forceinline__ void exch_wait_all(const Exch &e, uint64_t epoch) {
    const uint64_t *f = exch_flags(e.peers[e.rank]);
    SpinDeadline dl;
    for (int r = 0; r < e.world; ++r)  // no back-off: on the critical path of every fused collective
        while (ld_acquire_sys(f + r) < epoch) dl.spin("exchange: a peer never published its data");
}

// The last act of a call (one thread of the last block): this rank is done
// with `epoch` (its reads of its own area are complete and consumed) — written
// into every rank's area (relaxed: see above; the own copy is also the next
// call's epoch base) — and, for the NEXT call's stores, every rank has
// finished `epoch` - 1, whose parity buffer that call writes.  Bounded.
__device__ __forceinline__ void exch_finish(const Exch &e, uint64_t epoch) {
    for (int p = 0; p < e.world; ++p) st_relaxed_sys(exch_acks(e.peers[p]) + e.rank, epoch);
    const uint64_t *a = exch_acks(e.peers[e.rank]);
    SpinDeadline dl;
    for (int q = 0; q < e.world; ++q)
        while (ld_relaxed_sys(a + q) + 1ull < epoch) dl.pause("exchange: a peer never finished an earlier call");
}

}  // namespace lift
