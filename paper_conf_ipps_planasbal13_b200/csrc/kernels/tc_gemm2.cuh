// tc_gemm2.cuh — CTA-pair (cta_group::2) tcgen05 3xTF32 tile GEMM, sm_100a.
//
//   C[M x N] (ldc) = C + s * A[M x K] (lda) * op(B)        (same contract as tc_gemm.cuh)
//
// A cluster of two CTAs on one TPC computes a 256 x 256 output tile with UMMA M=256,
// N=256: CTA r of the pair stages rows [128r, 128r+128) of A and columns
// [128r, 128r+128) of B (big/small split, K-major SW128) in ITS shared memory; the leader
// (rank 0) issues tcgen05.mma.cta_group::2, which reads both CTAs' operands, and every
// CTA's TMEM receives its own 128 rows of the accumulator.  Per SM and per 32-wide k-block
// this stages 64 KB (vs 96 KB for one CTA at 128 x 256) and the tensor core reads 64 B/clk
// of shared memory instead of 96 B/clk, so the stage ring is 3 deep.
//   producers (warps 0-7 of each CTA): as tc_gemm (two k-blocks of loads in flight), then
//     fence.proxy.async and a cluster-scope arrive on the LEADER's full[s] barrier
//     (count 2 x 256); each CTA waits on its own empty[s], which the leader's
//     tcgen05.commit multicasts to both CTAs;
//   warp 8: TMEM allocation (cta_group::2, 512 columns: accumulator + staged C_in) in both
//     CTAs; MMA issue in the leader only;
//   epilogue: each CTA adds its C_in (TMEM columns [256, 512)) to its accumulator rows in
//     fp32 round-to-nearest and stores.
#pragma once
#include "tc_gemm.cuh"

namespace vsk {
namespace tc2 {

using namespace tc;

constexpr int BN2 = 256;        // pair tile N (each CTA stages 128 columns of B)
constexpr int BNH = BN2 / 2;
constexpr int STAGES2 = 3;
constexpr int A_BYTES2 = BM * BK * 4;     // 16 KB (this CTA's 128 rows)
constexpr int B_BYTES2 = BNH * BK * 4;    // 16 KB (this CTA's 128 columns)
constexpr int STAGE2 = 2 * A_BYTES2 + 2 * B_BYTES2;
constexpr int SMEM2 = STAGES2 * STAGE2 + 1024 + 256;
constexpr int APER2 = BM * BK / 4 / NPROD;    // 4 float4
constexpr int BPER2 = BNH * BK / 4 / NPROD;   // 4 float4

__device__ __forceinline__ uint32_t cluster_rank()
{
    uint32_t r;
    asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
    return r;
}
__device__ __forceinline__ void cluster_sync()
{
    asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
}
// arrive on the barrier at the same shared offset in CTA `target` of the cluster
__device__ __forceinline__ void mbar_arrive_cluster(uint64_t *bar, uint32_t target)
{
    uint32_t remote;
    asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(remote) : "r"(smem_u32(bar)), "r"(target));
    asm volatile("mbarrier.arrive.release.cluster.shared::cluster.b64 _, [%0];" ::"r"(remote) : "memory");
}
__device__ __forceinline__ void mbar_wait_cluster(uint64_t *bar, uint32_t parity)
{
    asm volatile(
        "{\n\t.reg .pred P1;\n"
        "WAIT_%=:\n\t"
        "mbarrier.try_wait.parity.acquire.cluster.shared::cta.b64 P1, [%0], %1;\n\t"
        "@P1 bra DONE_%=;\n\t"
        "bra WAIT_%=;\n"
        "DONE_%=:\n\t}" ::"r"(smem_u32(bar)),
        "r"(parity)
        : "memory");
}
__device__ __forceinline__ void mma_tf32_pair(uint32_t tmem_d, uint64_t adesc, uint64_t bdesc, uint32_t idesc, uint32_t acc)
{
    asm volatile(
        "{\n\t.reg .pred p;\n\t"
        "setp.ne.b32 p, %4, 0;\n\t"
        "tcgen05.mma.cta_group::2.kind::tf32 [%0], %1, %2, %3, p;\n\t}" ::"r"(tmem_d),
        "l"(adesc), "l"(bdesc), "r"(idesc), "r"(acc));
}
// commit the leader's MMAs to the barrier at this offset in BOTH CTAs of the pair
__device__ __forceinline__ void mma_commit_pair(uint64_t *bar)
{
    asm volatile(
        "tcgen05.commit.cta_group::2.mbarrier::arrive::one.shared::cluster.multicast::cluster.b64 [%0], %1;" ::"r"(
            smem_u32(bar)),
        "h"((uint16_t)0x3)
        : "memory");
}

template <bool NT, bool NEG, bool LOWER>
__global__ void __cluster_dims__(2, 1, 1) __launch_bounds__(NTHREADS, 1)
tc_gemm2_kernel(int M, int N, int K, const float *__restrict__ A, int lda, const float *__restrict__ B, int ldb,
                float *__restrict__ C, int ldc, TaskCtx ctx)
{
    ctx_begin(ctx);
    extern __shared__ uint8_t smem_raw[];
    // 1024-byte aligned, indexed from the __shared__ array so accesses stay LDS/STS
    uint8_t *smem = smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u);
    uint64_t *full = (uint64_t *)(smem + STAGES2 * STAGE2);
    uint64_t *empty = full + STAGES2;
    uint64_t *acc_full = empty + STAGES2;
    uint32_t *tmem_slot = (uint32_t *)(acc_full + 1);

    const uint32_t crank = cluster_rank();
    const int pair_m0 = (blockIdx.x & ~1) * BM;          // the pair's 256 rows
    const int m0 = pair_m0 + (int)crank * BM;            // this CTA's 128 rows
    const int n0 = blockIdx.y * BN2;                     // the pair's 256 columns
    const int nb0 = n0 + (int)crank * BNH;               // this CTA's 128 columns of B
    if (LOWER && n0 >= pair_m0 + 2 * BM) {               // whole pair tile above the diagonal
        ctx_end(ctx);
        return;
    }
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int nk = K / BK;

    if (threadIdx.x == 0) {
        for (int s = 0; s < STAGES2; s++) {
            mbar_init(&full[s], 2 * NPROD / 32);   // one arrive per producer warp of both CTAs
            mbar_init(&empty[s], 1);
        }
        mbar_init(acc_full, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    if (warp == NPROD / 32) {
        asm volatile("tcgen05.alloc.cta_group::2.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(tmem_slot)),
                     "r"(512u));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::2.sync.aligned;");
    }
    tc_fence_before();
    cluster_sync();                                      // barriers + TMEM of both CTAs ready
    tc_fence_after();
    const uint32_t tmem = *tmem_slot;

    if (warp < NPROD / 32) {
        const int t = threadIdx.x;
        const float4 z4 = make_float4(0.f, 0.f, 0.f, 0.f);
        auto load = [&](float4 (&ra)[APER2], float4 (&rb)[BPER2], int kb) {
            const int k0 = kb * BK;
#pragma unroll
            for (int p = 0; p < APER2; p++) {
                const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                ra[p] = (m0 + row < M) ? __ldg(reinterpret_cast<const float4 *>(A + (int64_t)(m0 + row) * lda + k0 + 4 * c)) : z4;
            }
            if (NT) {
#pragma unroll
                for (int p = 0; p < BPER2; p++) {
                    const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                    rb[p] = (nb0 + row < N) ? __ldg(reinterpret_cast<const float4 *>(B + (int64_t)(nb0 + row) * ldb + k0 + 4 * c)) : z4;
                }
            } else {
                const int u = t, kq = u / (BNH / 4), nq = u % (BNH / 4);   // one 4x4 unit per thread
                const bool ok = nb0 + 4 * nq < N;
#pragma unroll
                for (int i = 0; i < 4; i++)
                    rb[i] = ok ? __ldg(reinterpret_cast<const float4 *>(B + (int64_t)(k0 + 4 * kq + i) * ldb + nb0 + 4 * nq)) : z4;
            }
        };
        auto produce = [&](float4 (&ra)[APER2], float4 (&rb)[BPER2], int kb) {
            const int s = kb % STAGES2;
            if (kb >= STAGES2) mbar_wait(&empty[s], ((kb / STAGES2) - 1) & 1);
            uint8_t *st = smem + s * STAGE2;
            uint8_t *a_big = st, *a_small = st + A_BYTES2;
            uint8_t *b_big = st + 2 * A_BYTES2, *b_small = b_big + B_BYTES2;
#pragma unroll
            for (int p = 0; p < APER2; p++) {
                const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                store_split(a_big, a_small, kmaj_off(row, c), ra[p]);
            }
            if (NT) {
#pragma unroll
                for (int p = 0; p < BPER2; p++) {
                    const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                    store_split(b_big, b_small, kmaj_off(row, c), rb[p]);
                }
            } else {
                const int u = t, kq = u / (BNH / 4), nq = u % (BNH / 4);
                const float4 r0 = rb[0], r1 = rb[1], r2 = rb[2], r3 = rb[3];
                const int rot = (nq >> 1) & 3;
#pragma unroll
                for (int qq = 0; qq < 4; qq++) {
                    const int i = (qq + rot) & 3;
                    const float4 col = i == 0 ? make_float4(r0.x, r1.x, r2.x, r3.x)
                                     : i == 1 ? make_float4(r0.y, r1.y, r2.y, r3.y)
                                     : i == 2 ? make_float4(r0.z, r1.z, r2.z, r3.z)
                                              : make_float4(r0.w, r1.w, r2.w, r3.w);
                    store_split(b_big, b_small, kmaj_off(4 * nq + i, kq), col);
                }
            }
            fence_proxy_async();
            __syncwarp();
            if (lane == 0) mbar_arrive_cluster(&full[s], 0);      // the leader's barrier, one per warp
        };
        float4 ra0[APER2], rb0[BPER2], ra1[APER2], rb1[BPER2];
        load(ra0, rb0, 0);
        if (nk > 1) load(ra1, rb1, 1);
        // stage this CTA's C_in rows into TMEM columns [256, 512) (lane quarter eq, half eh)
        const int eq = warp & 3, eh = warp >> 2;
        const int erow = m0 + eq * 32 + lane;
#pragma unroll 1
        for (int c = 0; c < BN2 / 64; c++) {
            const int col0 = eh * (BN2 / 2) + c * 32;
            float v[32];
            const float *crow = C + (int64_t)erow * ldc + n0 + col0;
#pragma unroll
            for (int j = 0; j < 8; j++) {
                const float4 x = (erow < M && n0 + col0 + 4 * j < N) ? *reinterpret_cast<const float4 *>(crow + 4 * j) : z4;
                v[4 * j] = x.x; v[4 * j + 1] = x.y; v[4 * j + 2] = x.z; v[4 * j + 3] = x.w;
            }
            tmem_st32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)(BN2 + col0), v);
        }
        asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");
        for (int kb = 0; kb < nk; kb += 2) {
            produce(ra0, rb0, kb);
            if (kb + 2 < nk) load(ra0, rb0, kb + 2);
            if (kb + 1 < nk) {
                produce(ra1, rb1, kb + 1);
                if (kb + 3 < nk) load(ra1, rb1, kb + 3);
            }
        }
        // ---- epilogue: this CTA's 128 rows
        mbar_wait(acc_full, 0);
        tc_fence_after();
#pragma unroll 1
        for (int c = 0; c < BN2 / 64; c++) {
            const int col0 = eh * (BN2 / 2) + c * 32;
            float v[32], cv[32];
            tmem_ld32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)col0, v);
            tmem_ld32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)(BN2 + col0), cv);
#pragma unroll
            for (int i = 0; i < 32; i++) v[i] = cv[i] + v[i];
            if (erow < M) {
                float *crow = C + (int64_t)erow * ldc + n0 + col0;
#pragma unroll
                for (int j = 0; j < 8; j++) {
                    const int col = n0 + col0 + 4 * j;
                    if (col >= N) break;
                    if (LOWER && col + 3 > erow) {
                        if (col + 0 <= erow) crow[4 * j + 0] = v[4 * j + 0];
                        if (col + 1 <= erow) crow[4 * j + 1] = v[4 * j + 1];
                        if (col + 2 <= erow) crow[4 * j + 2] = v[4 * j + 2];
                    } else {
                        *reinterpret_cast<float4 *>(crow + 4 * j) =
                            make_float4(v[4 * j + 0], v[4 * j + 1], v[4 * j + 2], v[4 * j + 3]);
                    }
                }
            }
        }
    } else if (crank == 0) {
        // ---- MMA issuer (leader only): D[256 x 256] over both CTAs' operands
        constexpr uint32_t idesc = make_idesc(2 * BM, BN2, NEG, false);
        for (int kb = 0; kb < nk; kb++) {
            const int s = kb % STAGES2;
            mbar_wait_cluster(&full[s], (kb / STAGES2) & 1);
            tc_fence_after();
            if (lane == 0) {
                uint8_t *st = smem + s * STAGE2;
                const uint32_t a_big = smem_u32(st), a_small = a_big + A_BYTES2;
                const uint32_t b_big = a_big + 2 * A_BYTES2, b_small = b_big + B_BYTES2;
#pragma unroll
                for (int kk = 0; kk < BK / 8; kk++) {
                    const uint32_t o = kk * 32;
                    const uint64_t dAb = make_desc(a_big + o, 16, 1024), dAs = make_desc(a_small + o, 16, 1024);
                    const uint64_t dBb = make_desc(b_big + o, 16, 1024), dBs = make_desc(b_small + o, 16, 1024);
                    const uint32_t first = (kb == 0 && kk == 0) ? 0u : 1u;
                    mma_tf32_pair(tmem, dAb, dBb, idesc, first);
                    mma_tf32_pair(tmem, dAb, dBs, idesc, 1u);
                    mma_tf32_pair(tmem, dAs, dBb, idesc, 1u);
                }
                mma_commit_pair(&empty[s]);
                if (kb == nk - 1) mma_commit_pair(acc_full);
            }
            __syncwarp();
        }
    }

    tc_fence_before();
    cluster_sync();                                      // both CTAs done with TMEM / smem
    if (warp == NPROD / 32) {
        tc_fence_after();
        asm volatile("tcgen05.dealloc.cta_group::2.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"(512u));
    }
    ctx_end(ctx);
}

template <bool NT, bool NEG, bool LOWER>
inline int tc_gemm2(int M, int N, int K, const float *A, int lda, const float *B, int ldb, float *C, int ldc,
                    cudaStream_t s, const TaskCtx &ctx = TaskCtx())
{
    if (M <= 0 || N <= 0) return 0;
    if (K % BK) return -1;
    auto kern = tc_gemm2_kernel<NT, NEG, LOWER>;
    static bool attr[64] = {};
    int dev = 0;
    cudaGetDevice(&dev);
    if (!attr[dev & 63]) {
        cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, SMEM2);
        attr[dev & 63] = true;
    }
    int gx = (M + BM - 1) / BM;
    gx += gx & 1;                                        // whole CTA pairs
    dim3 grid(gx, (N + BN2 - 1) / BN2);
    count_launch();
    kern<<<grid, NTHREADS, SMEM2, s>>>(M, N, K, A, lda, B, ldb, C, ldc, ctx);
    return 0;
}

}  // namespace tc2
}  // namespace vsk
