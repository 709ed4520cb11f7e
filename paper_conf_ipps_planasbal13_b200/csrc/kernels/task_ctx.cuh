// task_ctx.cuh — device-side execution-time record of one task (a14, reading R17).
//
// Every kernel of a built-in version receives the task's TaskCtx.  The first thread of
// each CTA (or of each work unit of a persistent kernel) notes %globaltimer when it starts
// and, when it ends, folds [start, end] into the task's device slot (atomicMax of ~start,
// i.e. the minimum start, and of end); the last unit of every kernel (ticket) copies the
// current {~start, end} into the task's host-mapped slot and re-arms the ticket.  Kernels
// of one task run in stream order, so the host slot holds [first CTA start of the first
// kernel, last CTA end of the last kernel] once the task's completion event has fired:
// the time the task really occupied the GPU, without the time its launch waited in the
// stream queue (which CUDA events would include).  Slots are reset in bulk by the
// runtime before each drive (one cudaMemsetAsync), so no per-task reset is issued.
#pragma once
#include <stdint.h>

#include <mutex>
#include <unordered_map>

#include "kernels.hpp"

namespace vsk {

__device__ __forceinline__ unsigned long long globaltimer_ns()
{
    unsigned long long t;
    asm volatile("mov.u64 %0, %globaltimer;" : "=l"(t));
    return t;
}

// start of this CTA (thread 0), for its busy time
__device__ __forceinline__ unsigned long long &ctx_cta_start()
{
    __shared__ unsigned long long t0;
    return t0;
}

__device__ __forceinline__ void ctx_begin(const TaskCtx &c)
{
    // (slot[0] keeps ~start so that max(~t) == min(t) and an all-zero slot is "empty")
    if (c.slot && threadIdx.x == 0) ctx_cta_start() = globaltimer_ns();
}

// Dependence release of a completed task (a3), by one full warp: decrement every successor's
// in-degree; the successors that became ready are appended to the ready ring with one
// warp-aggregated ticket per 32 successors.
__device__ __forceinline__ void ctx_release(const TaskCtx &c)
{
    const DevTracker *t = c.trk;
    const unsigned lane = threadIdx.x & 31u;
    const int b = t->succ_off[c.tidx], e = t->succ_off[c.tidx + 1];
    for (int i = b; i < e; i += 32) {
        int s = -1;
        if (i + (int)lane < e) {
            s = t->succ[i + lane];
            if (atomicSub(&t->indeg[s], 1) != 1) s = -1;
        }
        const unsigned m = __ballot_sync(0xffffffffu, s >= 0);
        if (!m) continue;
        const int leader = __ffs(m) - 1;
        unsigned long long pos = 0;
        if ((int)lane == leader) {
            __threadfence_system();   // the task's records and completion entry are visible first
            pos = atomicAdd(t->rdy_ctr, (unsigned long long)__popc(m));
        }
        pos = __shfl_sync(0xffffffffu, pos, leader);
        if (s >= 0) {
            pos += __popc(m & ((1u << lane) - 1u));
            volatile unsigned long long *r = t->rdy_ring;
            r[pos & (kRingCap - 1)] = (t->epoch << 32) | (unsigned long long)(s + 1);
        }
    }
}

// One work unit of the task finished (a CTA, or one output tile of a persistent kernel):
// [t0, t1] on %globaltimer.  Called by ONE thread after the unit's global stores (fenced).
// The unit that completes the task's count (ncta units per kernel) publishes the kernel's
// record; returns true when that was the task's last kernel and its successors are to be
// released (device tracker, a3) — the caller then runs ctx_release with a full warp.
__device__ __forceinline__ bool ctx_done(const TaskCtx &c, unsigned long long t0, unsigned long long t1,
                                         unsigned long long nct)
{
    bool release_now = false;
    atomicMax(&c.slot[0], ~t0);
    atomicMax(&c.slot[1], t1);
    const unsigned long long dur = t1 - t0;
    atomicAdd(&c.slot[3], dur);   // unit busy time
    atomicMax(&c.slot[4], dur);   // longest unit
    if (atomicAdd(&c.slot[2], 1ull) == nct - 1) {
        __threadfence();
        const unsigned long long s = atomicAdd(&c.slot[0], 0ull), e = atomicAdd(&c.slot[1], 0ull);
        const unsigned long long busy = atomicExch(&c.slot[3], 0ull), longest = atomicExch(&c.slot[4], 0ull);
        if (c.host) {
            volatile unsigned long long *h = c.host;
            h[0] = s;
            h[1] = e;
            // the kernel's execution time with the GPU to itself (reading R17): its
            // longest unit when all its units are resident at once (nsm x occ CTA slots),
            // else the units' summed busy time / CTA slots (waves)
            const unsigned long long slots = (unsigned long long)c.nsm * (c.occ ? c.occ : 1u);
            h[3] = h[3] + ((c.nsm && nct > slots) ? busy / slots : longest);
            // kernels of the task completed so far: the host polls this word (compared
            // with the number of kernels the version launched) instead of querying events
            __threadfence_system();
            h[2] = h[2] + 1;
            if (c.ring) {   // the record above is visible before the ring entry
                __threadfence_system();
                const unsigned long long pos = atomicAdd(c.ring_ctr, 1ull);
                volatile unsigned long long *r = c.ring;
                r[pos & (kRingCap - 1)] = c.tag;
            }
        }
        // the task's last kernel releases its successors (a3): kernels done on the device
        if (c.trk && atomicAdd(&c.slot[5], 1ull) + 1 == (unsigned long long)c.nkern) release_now = true;
        atomicExch(&c.slot[2], 0ull);   // re-arm for the task's next kernel
    }
    return release_now;
}

// Call once per CTA, by all threads of the CTA, on every exit path (after the CTA's
// last global store).
__device__ __forceinline__ void ctx_end(const TaskCtx &c)
{
    if (!c.slot) return;
    __shared__ int release_now;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        const unsigned long long nct = c.ncta ? (unsigned long long)c.ncta
                                              : (unsigned long long)gridDim.x * gridDim.y * gridDim.z;
        release_now = ctx_done(c, ctx_cta_start(), globaltimer_ns(), nct) ? 1 : 0;
    }
    if (c.trk) {
        __syncthreads();
        if (release_now && threadIdx.x < 32) ctx_release(c);
    }
}

__global__ void __launch_bounds__(32) release_kernel(const TaskCtx c)
{
    ctx_release(c);
}

// Resident CTAs per SM of `kernel` at (threads, dynamic smem) on the current device, cached
// per kernel; the launch sites put it in the task's TaskCtx (execution-time measure, R17).
template <class K>
unsigned kernel_occupancy(K kernel, int threads, size_t smem)
{
    static std::mutex mu;
    static std::unordered_map<const void *, unsigned> cache;
    std::lock_guard<std::mutex> lock(mu);
    auto it = cache.find((const void *)kernel);
    if (it != cache.end()) return it->second;
    int n = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&n, kernel, threads, smem) != cudaSuccess || n < 1) {
        cudaGetLastError();
        n = 1;
    }
    cache[(const void *)kernel] = (unsigned)n;
    return (unsigned)n;
}

template <class K>
TaskCtx ctx_for(const TaskCtx &c, K kernel, int threads, size_t smem)
{
    TaskCtx x = c;
    if (x.slot) x.occ = kernel_occupancy(kernel, threads, smem);
    return x;
}

}  // namespace vsk
