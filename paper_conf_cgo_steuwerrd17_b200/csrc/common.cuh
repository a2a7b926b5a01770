// common.cuh — sm_100a device helpers shared by the Lift hot-path kernels.
//
// Vocabulary follows the paper (Sec. 3.2):
//   reduceSeq  (L320)      per-thread sequential fold in registers
//   iterate    (L312-324)  the in-block tree (here: warp butterfly + smem)
//   toLocal    (L368-377)  shared memory; toPrivate = registers
//   asVector4  (L378-389)  128-bit float4 accesses
#pragma once

#include <cuda_runtime.h>
#include <stdint.h>
#include <stdlib.h>

#include <mutex>

namespace lift {

constexpr int kWarp = 32;

// ---------------------------------------------------------------------------
// Bounded spins.  Every in-kernel wait on another block or rank (grid barrier,
// exchange flags) gives up after a time limit and traps (the launch fails with
// an error at the caller's next synchronisation) instead of hanging the GPU
// when its partner can never arrive: blocks that are not co-resident, a peer
// rank that never makes the matching call.  The limit (default 20 s, far above
// any legitimate wait: the slowest kernel here takes ~3 ms) comes from
// LIFT_SPIN_TIMEOUT_MS, read when the library first touches a device.
// ---------------------------------------------------------------------------
constexpr unsigned long long kSpinLimitDefaultNs = 20ull * 1000 * 1000 * 1000;
static __device__ unsigned long long g_spin_limit_ns = kSpinLimitDefaultNs;  // one copy per translation unit

__device__ __forceinline__ unsigned long long globaltimer_ns() {
    unsigned long long t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    return t;
}

struct SpinDeadline {
    unsigned long long t0 = 0;
    unsigned int polls = 0;
    // trap once the limit has passed since the first call
    __device__ __forceinline__ void check(const char * /* what is awaited (documentation) */) {
        const unsigned long long t = globaltimer_ns();
        if (t0 == 0)
            t0 = t;
        else if (t - t0 > g_spin_limit_ns)
            __trap();
    }
    // one failed poll: back off, then check the deadline
    __device__ __forceinline__ void pause(const char *what, unsigned ns = 64) {
        __nanosleep(ns);
        check(what);
    }
    // one failed poll of a latency-critical wait: no back-off, the deadline
    // checked every 256 polls
    __device__ __forceinline__ void spin(const char *what) {
        if ((++polls & 255u) == 0) check(what);
    }
};

static inline unsigned long long spin_limit_from_env() {
    const char *v = getenv("LIFT_SPIN_TIMEOUT_MS");
    if (v == nullptr || *v == 0) return kSpinLimitDefaultNs;
    const long long ms = atoll(v);
    return ms > 0 ? (unsigned long long)ms * 1000000ull : kSpinLimitDefaultNs;
}
// sets this translation unit's copy on the current device
static inline cudaError_t set_spin_limit_here() {
    const unsigned long long ns = spin_limit_from_env();
    return cudaMemcpyToSymbol(g_spin_limit_ns, &ns, sizeof ns);
}

// ---------------------------------------------------------------------------
// Host-side launch helpers, cached per (kernel, device, shape): the CUDA
// queries cost ~1-3 us of host time each, more than a small launch itself.
// ---------------------------------------------------------------------------
struct KernelCache {
    struct Entry {
        const void *kern;
        int dev, threads;
        size_t smem;
        int value;
    };
    Entry e[256];
    int used = 0;
    std::mutex mu;
};
static inline KernelCache &kernel_cache() {
    static KernelCache c;  // one per translation unit is enough (keys include the kernel)
    return c;
}
// cudaOccupancyMaxActiveBlocksPerMultiprocessor, cached
template <typename K>
static inline cudaError_t occupancy_cached(K kern, int dev, int threads, size_t smem, int *per_sm) {
    KernelCache &c = kernel_cache();
    const void *kp = reinterpret_cast<const void *>(kern);
    {
        std::lock_guard<std::mutex> lock(c.mu);
        for (int i = 0; i < c.used; ++i)
            if (c.e[i].kern == kp && c.e[i].dev == dev && c.e[i].threads == threads && c.e[i].smem == smem) {
                *per_sm = c.e[i].value;
                return cudaSuccess;
            }
    }
    cudaError_t err = cudaOccupancyMaxActiveBlocksPerMultiprocessor(per_sm, kern, threads, smem);
    if (err != cudaSuccess) return err;
    std::lock_guard<std::mutex> lock(c.mu);
    if (c.used < 256) c.e[c.used++] = KernelCache::Entry{kp, dev, threads, smem, *per_sm};
    return cudaSuccess;
}
// cudaFuncAttributeMaxDynamicSharedMemorySize >= smem, set once per (kernel, device)
template <typename K>
static inline cudaError_t ensure_smem(K kern, int dev, size_t smem) {
    if (smem <= 48 * 1024) return cudaSuccess;
    KernelCache &c = kernel_cache();
    const void *kp = reinterpret_cast<const void *>(kern);
    std::lock_guard<std::mutex> lock(c.mu);
    for (int i = 0; i < c.used; ++i)
        if (c.e[i].kern == kp && c.e[i].dev == dev && c.e[i].threads == -1) {
            if (c.e[i].smem >= smem) return cudaSuccess;
            cudaError_t err = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
            if (err == cudaSuccess) c.e[i].smem = smem;
            return err;
        }
    cudaError_t err = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (err == cudaSuccess && c.used < 256) c.e[c.used++] = KernelCache::Entry{kp, dev, -1, smem, 0};
    return err;
}

// ---------------------------------------------------------------------------
// Programmatic dependent launch (PDL): the streaming kernels are launched with
// cudaLaunchAttributeProgrammaticStreamSerialization, so the next kernel on the
// stream can be scheduled onto SMs as this one's blocks retire; each kernel
// starts with griddepcontrol.wait (before ANY global memory access: the
// previous kernel may produce its inputs or read its outputs) and then lets
// its own dependent launch.  The cooperative fused ATAX kernels take the same
// attribute beside their cooperative / cluster ones but never trigger early
// (atax.cu); the fused collectives do not take it (launch_pdl's `allow`).
// LIFT_PDL=0 turns it off (A/B).
// ---------------------------------------------------------------------------
__device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;" ::: "memory"); }
// Before its griddepcontrol.wait a dependent block may already pull the first
// bytes of its READ-ONLY stream into L2 (cp.async.bulk.prefetch.L2, issued
// while the previous kernel drains).  A prefetch returns nothing to the
// program and L2 is the device's point of coherence, so even a range the
// previous kernel is still writing cannot be read stale: only the loads after
// pdl_wait() deliver data.  -DLIFT_PDL_PREFETCH=0 compiles it out (A/B).
#ifndef LIFT_PDL_PREFETCH
#define LIFT_PDL_PREFETCH 1
#endif
__device__ __forceinline__ void pdl_release() { asm volatile("griddepcontrol.launch_dependents;" ::: "memory"); }
__device__ __forceinline__ void pdl_wait_and_release() {
    pdl_wait();
    pdl_release();
}
static inline bool pdl_enabled() {
    static const bool on = [] {
        const char *v = getenv("LIFT_PDL");
        return !(v && v[0] == '0');
    }();
    return on;
}
// kern<<<grid, block, smem, s>>>(args...) with the PDL attribute (unless `allow` is
// false: the fused collectives launch plainly — a dependent's early blocks could
// take SM slots a peer rank SHARING the GPU needs before this kernel can finish)
template <typename... KArgs, typename... Args>
static inline cudaError_t launch_pdl(bool allow, void (*kern)(KArgs...), dim3 grid, dim3 block, size_t smem,
                                     cudaStream_t s, Args &&...args) {
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    attr[0].val.programmaticStreamSerializationAllowed = (allow && pdl_enabled()) ? 1 : 0;
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = grid;
    cfg.blockDim = block;
    cfg.dynamicSmemBytes = smem;
    cfg.stream = s;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    return cudaLaunchKernelEx(&cfg, kern, static_cast<KArgs>(args)...);
}

// ---------------------------------------------------------------------------
// Global loads
// ---------------------------------------------------------------------------

// Streaming 128-bit read-only load: the big operand (A, B, x/y of dot) is
// touched exactly once, so do not allocate it in L1.
__device__ __forceinline__ float4 ld_stream4(const float4 *p) {
    float4 r;
    asm volatile("ld.global.nc.L1::no_allocate.v4.f32 {%0,%1,%2,%3}, [%4];"
                 : "=f"(r.x), "=f"(r.y), "=f"(r.z), "=f"(r.w)
                 : "l"(p));
    return r;
}

__device__ __forceinline__ float ld_stream1(const float *p) {
    float r;
    asm volatile("ld.global.nc.L1::no_allocate.f32 %0, [%1];" : "=f"(r) : "l"(p));
    return r;
}

// Read-only cached loads for small operands reused by many threads (x, t).
__device__ __forceinline__ float4 ld_ro4(const float4 *p) { return __ldg(p); }
__device__ __forceinline__ float ld_ro1(const float *p) { return __ldg(p); }

// ---------------------------------------------------------------------------
// multAndSumUp (L767, Fig. 7 l.12 = L959): acc + a*b with one rounding (FMA)
// — reading R2 — applied per float4 component (mapVec, L381-383).
// ---------------------------------------------------------------------------
__device__ __forceinline__ void fma4(float4 &acc, const float4 a, const float4 b) {
    acc.x = __fmaf_rn(a.x, b.x, acc.x);
    acc.y = __fmaf_rn(a.y, b.y, acc.y);
    acc.z = __fmaf_rn(a.z, b.z, acc.z);
    acc.w = __fmaf_rn(a.w, b.w, acc.w);
}

__device__ __forceinline__ void fma4s(float4 &acc, const float4 a, const float s) {
    acc.x = __fmaf_rn(a.x, s, acc.x);
    acc.y = __fmaf_rn(a.y, s, acc.y);
    acc.z = __fmaf_rn(a.z, s, acc.z);
    acc.w = __fmaf_rn(a.w, s, acc.w);
}

// Fixed-shape fold of the four component accumulators: (x + y) + (z + w).
__device__ __forceinline__ float hsum4(const float4 v) {
    return __fadd_rn(__fadd_rn(v.x, v.y), __fadd_rn(v.z, v.w));
}

// GPU-scope release / acquire-release counters (PTX memory model).  A block
// publishes its partial with ONE release operation after a block barrier
// (cumulativity covers the other threads' stores), instead of
// __threadfence() + atomicAdd: __threadfence is fence.sc (MEMBAR.SC.GPU plus an
// L1 invalidate), stronger than the release these hand-offs need.
__device__ __forceinline__ void red_release_add(unsigned int *p, unsigned int v) {
    asm volatile("red.release.gpu.global.add.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ unsigned int atom_acq_rel_add(unsigned int *p, unsigned int v) {
    unsigned int r;
    asm volatile("atom.acq_rel.gpu.global.add.u32 %0, [%1], %2;" : "=r"(r) : "l"(p), "r"(v) : "memory");
    return r;
}
__device__ __forceinline__ unsigned int ld_acquire_gpu(const unsigned int *p) {
    unsigned int v;
    asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
    return v;
}

// Drop one 128-byte L2 line without writing it back (PTX discard.global.L2).
// Used on partial-sum rows once their only reader has consumed them: the next
// launch rewrites them, so their dirty lines would otherwise cost a DRAM
// write-back in the middle of the next stream (~1 us per 4.8 MB at 8192^2).
__device__ __forceinline__ void discard_l2_line(const void *p) {
    asm volatile("discard.global.L2 [%0], 128;" ::"l"(p) : "memory");
}

__device__ __forceinline__ float4 zero4() { return make_float4(0.f, 0.f, 0.f, 0.f); }

// ---------------------------------------------------------------------------
// In-warp tree (the iterate-over-local-memory step of Listing 1,
// done with register shuffles instead of local memory + barriers, Sec. 5.4).
// Butterfly: every lane ends with the same bits (fp add is commutative).
// ---------------------------------------------------------------------------
__device__ __forceinline__ float warp_sum(float v) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v = __fadd_rn(v, __shfl_xor_sync(0xffffffffu, v, o));
    return v;
}

// Pairwise (adjacent) tree over a power-of-two number of values in order:
// out = ((v0+v1)+(v2+v3)) + ...  — Listing 1's iterate over split2.
template <int N>
__device__ __forceinline__ float pair_tree(const float *v) {
    if constexpr (N == 1) {
        return v[0];
    } else {
        float t[N / 2];
#pragma unroll
        for (int i = 0; i < N / 2; ++i) t[i] = __fadd_rn(v[2 * i], v[2 * i + 1]);
        return pair_tree<N / 2>(t);
    }
}

// ---------------------------------------------------------------------------
// mbarrier + 1-D bulk copy (TMA engine; SASS UBLKCP) for staging x in smem.
// ---------------------------------------------------------------------------
__device__ __forceinline__ uint32_t smem_u32(const void *p) {
    return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}

// CTA-scope acquire-release add on a shared-memory counter ("last arriver" hand-offs)
__device__ __forceinline__ unsigned int atom_acq_rel_add_cta_shared(unsigned int *p, unsigned int v) {
    unsigned int r;
    asm volatile("atom.acq_rel.cta.shared::cta.add.u32 %0, [%1], %2;" : "=r"(r) : "r"(smem_u32(p)), "r"(v) : "memory");
    return r;
}

__device__ __forceinline__ void mbar_init(uint64_t *bar, uint32_t count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count));
}

__device__ __forceinline__ void fence_mbar_init() {
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}

__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t *bar, uint32_t bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
                 : "memory");
}

__device__ __forceinline__ void mbar_wait_parity(uint64_t *bar, uint32_t parity) {
    asm volatile(
        "{\n"
        ".reg .pred p;\n"
        "LIFT_WAIT_%=:\n"
        "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n"
        "@!p bra LIFT_WAIT_%=;\n"
        "}\n" ::"r"(smem_u32(bar)),
        "r"(parity)
        : "memory");
}

// global -> shared bulk copy; bytes % 16 == 0, both addresses 16-B aligned.
__device__ __forceinline__ void bulk_g2s(void *dst_smem, const void *src_gmem, uint32_t bytes, uint64_t *bar) {
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
            smem_u32(dst_smem)),
        "l"(src_gmem), "r"(bytes), "r"(smem_u32(bar))
        : "memory");
}

// The same with an L2 eviction-priority hint: `policy` from l2_policy_evict_first()
// marks the streamed lines as the first to go, so a single-use stream does not
// push the kernel's own instructions and small reused data out of L2.
__device__ __forceinline__ uint64_t l2_policy_evict_first() {
    uint64_t pol;
    asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(pol));
    return pol;
}
__device__ __forceinline__ void bulk_g2s_hint(void *dst_smem, const void *src_gmem, uint32_t bytes, uint64_t *bar,
                                              uint64_t policy) {
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1], %2, [%3], "
        "%4;" ::"r"(smem_u32(dst_smem)),
        "l"(src_gmem), "r"(bytes), "r"(smem_u32(bar)), "l"(policy)
        : "memory");
}

// Prefetch `bytes` (multiple of 16) of gmem into L2 with the bulk-copy engine
// (no smem, no completion tracking).
__device__ __forceinline__ void bulk_prefetch_l2(const void *src_gmem, uint32_t bytes) {
    asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(src_gmem), "r"(bytes) : "memory");
}

// Stage `bytes` (multiple of 16) of gmem into smem with the bulk-copy engine.
// Called by ALL threads of the block; thread 0 issues. Returns after the data
// has landed (mbarrier phase 0 completes).  `bar` must be a fresh mbarrier
// slot in shared memory.  Work independent of the staged data may be issued
// by the caller before calling stage_wait().
__device__ __forceinline__ void stage_issue(void *dst, const void *src, uint32_t bytes, uint64_t *bar) {
    if (threadIdx.x == 0) {
        mbar_init(bar, 1);
        fence_mbar_init();
    }
    __syncthreads();
    if (threadIdx.x == 0) {
        mbar_arrive_expect_tx(bar, bytes);
        constexpr uint32_t kChunk = 32768;
        for (uint32_t off = 0; off < bytes; off += kChunk) {
            uint32_t b = bytes - off < kChunk ? bytes - off : kChunk;
            bulk_g2s(static_cast<char *>(dst) + off, static_cast<const char *>(src) + off, b, bar);
        }
    }
}

__device__ __forceinline__ void stage_wait(uint64_t *bar) { mbar_wait_parity(bar, 0); }

// ---------------------------------------------------------------------------
// Thread-block clusters: rank / id registers, split cluster barrier, and
// distributed shared memory (DSMEM) loads/stores of a peer block's smem.
// ---------------------------------------------------------------------------
__device__ __forceinline__ uint32_t cluster_ctarank() {
    uint32_t r;
    asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
    return r;
}
__device__ __forceinline__ uint32_t cluster_nctarank() {
    uint32_t r;
    asm volatile("mov.u32 %0, %%cluster_nctarank;" : "=r"(r));
    return r;
}
__device__ __forceinline__ uint32_t cluster_id_x() {
    uint32_t r;
    asm volatile("mov.u32 %0, %%clusterid.x;" : "=r"(r));
    return r;
}
__device__ __forceinline__ uint32_t cluster_count_x() {
    uint32_t r;
    asm volatile("mov.u32 %0, %%nclusterid.x;" : "=r"(r));
    return r;
}
__device__ __forceinline__ void cluster_arrive() {
    asm volatile("barrier.cluster.arrive.release.aligned;" ::: "memory");
}
__device__ __forceinline__ void cluster_wait() { asm volatile("barrier.cluster.wait.acquire.aligned;" ::: "memory"); }
__device__ __forceinline__ void cluster_sync() {
    cluster_arrive();
    cluster_wait();
}
// address of the same smem variable in block `rank` of this cluster
__device__ __forceinline__ uint32_t dsmem_addr(const void *local, uint32_t rank) {
    uint32_t a;
    asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(a) : "r"(smem_u32(local)), "r"(rank));
    return a;
}
__device__ __forceinline__ uint32_t dsmem_addr_raw(uint32_t local_smem, uint32_t rank) {
    uint32_t a;
    asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(a) : "r"(local_smem), "r"(rank));
    return a;
}
// Asynchronous remote store that completes `4` transaction bytes on the
// destination CTA's mbarrier when the value lands (no membar needed).
__device__ __forceinline__ void st_async_dsmem1(uint32_t addr, float v, uint32_t remote_bar) {
    asm volatile("st.async.shared::cluster.mbarrier::complete_tx::bytes.b32 [%0], %1, [%2];" ::"r"(addr),
                 "r"(__float_as_uint(v)), "r"(remote_bar)
                 : "memory");
}
__device__ __forceinline__ void st_dsmem1(uint32_t addr, float v) {
    asm volatile("st.shared::cluster.f32 [%0], %1;" ::"r"(addr), "f"(v) : "memory");
}
__device__ __forceinline__ float4 ld_dsmem4(uint32_t addr) {
    float4 v;
    asm volatile("ld.shared::cluster.v4.f32 {%0, %1, %2, %3}, [%4];"
                 : "=f"(v.x), "=f"(v.y), "=f"(v.z), "=f"(v.w)
                 : "r"(addr)
                 : "memory");
    return v;
}

// Named barrier over `nthreads` threads (multiple of 32) with id in [1, 15].
__device__ __forceinline__ void named_bar_sync(int id, int nthreads) {
    asm volatile("bar.sync %0, %1;" ::"r"(id), "r"(nthreads) : "memory");
}

}  // namespace lift
