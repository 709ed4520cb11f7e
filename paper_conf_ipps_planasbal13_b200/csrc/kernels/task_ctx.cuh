// task_ctx.cuh — device-side execution-time record of one task (a14, reading R17).
//
// Every kernel of a built-in version receives the task's TaskCtx.  The first thread of
// each CTA folds %globaltimer into the task's device slot when the CTA starts
// (atomicMax of ~t, i.e. the minimum start) and ends (atomicMax); the last CTA of every
// kernel (ticket) copies the current {~start, end} into the task's host-mapped slot and
// re-arms the ticket.  Kernels
// of one task run in stream order, so the host slot holds [first CTA start of the first
// kernel, last CTA end of the last kernel] once the task's completion event has fired:
// the time the task really occupied the GPU, without the time its launch waited in the
// stream queue (which CUDA events would include).  Slots are reset in bulk by the
// runtime before each drive (one cudaMemsetAsync), so no per-task reset is issued.
#pragma once
#include <stdint.h>

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
    // slot[0] keeps ~start so that max(~t) == min(t) and an all-zero slot is "empty"
    if (c.slot && threadIdx.x == 0) {
        const unsigned long long t = globaltimer_ns();
        ctx_cta_start() = t;
        atomicMax(&c.slot[0], ~t);
    }
}

// Call once per CTA, by all threads of the CTA, on every exit path (after the CTA's
// last global store).
__device__ __forceinline__ void ctx_end(const TaskCtx &c)
{
    if (!c.slot) return;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        const unsigned long long t = globaltimer_ns();
        atomicMax(&c.slot[1], t);
        const unsigned long long dur = t - ctx_cta_start();
        atomicAdd(&c.slot[3], dur);   // CTA busy time
        atomicMax(&c.slot[4], dur);   // longest CTA
        const unsigned long long nct = c.ncta ? (unsigned long long)c.ncta
                                              : (unsigned long long)gridDim.x * gridDim.y * gridDim.z;
        if (atomicAdd(&c.slot[2], 1ull) == nct - 1) {
            __threadfence();
            const unsigned long long s = atomicAdd(&c.slot[0], 0ull), e = atomicAdd(&c.slot[1], 0ull);
            const unsigned long long busy = atomicExch(&c.slot[3], 0ull), longest = atomicExch(&c.slot[4], 0ull);
            if (c.host) {
                volatile unsigned long long *h = c.host;
                h[0] = s;
                h[1] = e;
                // the kernel's execution time with the GPU to itself (reading R17): its
                // longest CTA when all CTAs fit at once (one per SM), else CTA busy time / SMs
                h[3] = h[3] + ((c.nsm && nct > c.nsm) ? busy / c.nsm : longest);
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
            atomicExch(&c.slot[2], 0ull);   // re-arm for the task's next kernel
        }
    }
}

}  // namespace vsk
