// tc_gemm.cuh — tcgen05 / TMEM 3xTF32 tile GEMM (version tc_3xtf32), sm_100a.
//
//   C[M x N] (ldc) = C + s * A[M x K] (lda) * op(B),  s = +1 (matmul) or -1 (Cholesky
//   gemm / syrk / trsm / potrf updates), op(B) = B (NN) or B^T (NT).
//
// 3xTF32: every fp32 operand x is split into big = rna_tf32(x) and small = x - big
// (exact in fp32), and D += Ab*Bb + Ab*Bs + As*Bb is accumulated in fp32 in TMEM by
// three tcgen05.mma.kind::tf32 per 8-wide k-step (the dropped As*Bs term is
// < 2^-22 |a||b|).  The sign s is the instruction descriptor's negate-A bit.
//
// Structure (one 128 x BN output tile per CTA, cta_group::1, UMMA M=128, N=BN):
//   warps 0-7  producers (256 threads): LDG.128 of fp32 k-blocks (32 wide) two k-blocks
//              ahead in registers -> split -> STS.128 into 128B-swizzled K-major UMMA
//              layouts (A; B in NT form; B in NN form after a 4x4 register transpose so
//              the store stays a conflict-free 16-byte vector) -> fence.proxy.async ->
//              mbarrier arrive (full[s]).  STAGES smem stages of {A,B} x {big,small}.
//   warp 8     TMEM allocator + MMA issuer: one lane waits full[s], issues 3 x (BK/8)
//              tcgen05.mma, tcgen05.commit -> empty[s]; after the last k-block,
//              commit -> acc_full.
//   warps 0-7  C_in prefetch: before the main loop each producer warp copies its part of
//              the C tile (TMEM lanes 32(w%4).., column half w/4) into TMEM columns
//              [BN, 2BN) with tcgen05.st, overlapping the first operand loads.
//   warps 0-7  epilogue: tcgen05.ld of the accumulator and of C_in, C = C_in + acc in fp32
//              round-to-nearest, vector stores (no global loads in the epilogue).
// LOWER (syrk / potrf update): CTAs strictly above the diagonal exit; diagonal tiles
// store only j <= i.
// The MN-major B encoding (no transpose) was probed on B200 (tools/probe_mn.cu): with the
// B-major bit set the tf32 MMA contributed nothing, so NN B is transposed in registers.
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include "kernels.hpp"
#include "task_ctx.cuh"

namespace vsk {
namespace tc {

constexpr int BM = 128, BK = 32;
constexpr int kKChunk = 1024;   // largest K accumulated in TMEM by one launch (see tc_gemm)
constexpr int NPROD = 256;  // producer / epilogue threads (warps 0-7)
constexpr int NTHREADS = NPROD + 32;

__device__ __forceinline__ uint32_t smem_u32(const void *p) { return (uint32_t)__cvta_generic_to_shared(p); }

__device__ __forceinline__ void mbar_init(uint64_t *bar, uint32_t count)
{
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count));
}
__device__ __forceinline__ void mbar_arrive(uint64_t *bar)
{
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
__device__ __forceinline__ void mbar_wait(uint64_t *bar, uint32_t parity)
{
    asm volatile(
        "{\n\t.reg .pred P1;\n"
        "WAIT_%=:\n\t"
        "mbarrier.try_wait.parity.shared::cta.b64 P1, [%0], %1;\n\t"
        "@P1 bra DONE_%=;\n\t"
        "bra WAIT_%=;\n"
        "DONE_%=:\n\t}" ::"r"(smem_u32(bar)),
        "r"(parity)
        : "memory");
}
__device__ __forceinline__ void fence_proxy_async() { asm volatile("fence.proxy.async.shared::cta;" ::: "memory"); }
__device__ __forceinline__ void tc_fence_before() { asm volatile("tcgen05.fence::before_thread_sync;" ::: "memory"); }
__device__ __forceinline__ void tc_fence_after() { asm volatile("tcgen05.fence::after_thread_sync;" ::: "memory"); }

__device__ __forceinline__ float to_tf32(float x)
{
    uint32_t r;
    asm("cvt.rna.tf32.f32 %0, %1;" : "=r"(r) : "f"(x));
    return __uint_as_float(r);
}

// UMMA shared-memory descriptor (sm_100): start>>4 [0,14), LBO>>4 [16,30), SBO>>4 [32,46),
// version=1 [46,48), base offset 0, layout SWIZZLE_128B = 2 at [61,64).
__device__ __forceinline__ uint64_t make_desc(uint32_t saddr, uint32_t lbo, uint32_t sbo)
{
    uint64_t d = 0;
    d |= (uint64_t)((saddr & 0x3FFFF) >> 4);
    d |= (uint64_t)((lbo >> 4) & 0x3FFF) << 16;
    d |= (uint64_t)((sbo >> 4) & 0x3FFF) << 32;
    d |= (uint64_t)1 << 46;
    d |= (uint64_t)2 << 61;
    return d;
}

// Instruction descriptor, kind::tf32: D f32 (bit 4), A/B tf32 (=2 at bits 7, 10),
// negate A (bit 13), B major (bit 16: 1 = MN-major), N>>3 at 17, M>>4 at 24.
__host__ __device__ constexpr uint32_t make_idesc(int M, int N, bool negA, bool b_mn_major)
{
    return (1u << 4) | (2u << 7) | (2u << 10) | ((negA ? 1u : 0u) << 13) | ((b_mn_major ? 1u : 0u) << 16) |
           ((uint32_t)(N >> 3) << 17) | ((uint32_t)(M >> 4) << 24);
}

__device__ __forceinline__ void mma_tf32(uint32_t tmem_d, uint64_t adesc, uint64_t bdesc, uint32_t idesc, uint32_t acc)
{
    asm volatile(
        "{\n\t.reg .pred p;\n\t"
        "setp.ne.b32 p, %4, 0;\n\t"
        "tcgen05.mma.cta_group::1.kind::tf32 [%0], %1, %2, %3, p;\n\t}" ::"r"(tmem_d),
        "l"(adesc), "l"(bdesc), "r"(idesc), "r"(acc));
}
__device__ __forceinline__ void mma_commit(uint64_t *bar)
{
    asm volatile("tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.b64 [%0];" ::"r"(smem_u32(bar))
                 : "memory");
}

__device__ __forceinline__ void tmem_st32(uint32_t taddr, const float (&v)[32])
{
    asm volatile(
        "tcgen05.st.sync.aligned.32x32b.x32.b32 [%0], {%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15,%16,"
        "%17,%18,%19,%20,%21,%22,%23,%24,%25,%26,%27,%28,%29,%30,%31,%32};" ::"r"(taddr),
        "f"(v[0]), "f"(v[1]), "f"(v[2]), "f"(v[3]), "f"(v[4]), "f"(v[5]), "f"(v[6]), "f"(v[7]), "f"(v[8]), "f"(v[9]),
        "f"(v[10]), "f"(v[11]), "f"(v[12]), "f"(v[13]), "f"(v[14]), "f"(v[15]), "f"(v[16]), "f"(v[17]), "f"(v[18]),
        "f"(v[19]), "f"(v[20]), "f"(v[21]), "f"(v[22]), "f"(v[23]), "f"(v[24]), "f"(v[25]), "f"(v[26]), "f"(v[27]),
        "f"(v[28]), "f"(v[29]), "f"(v[30]), "f"(v[31])
        : "memory");
}

__device__ __forceinline__ void tmem_ld32(uint32_t taddr, float (&v)[32])
{
    uint32_t r[32];
    asm volatile(
        "tcgen05.ld.sync.aligned.32x32b.x32.b32 {%0,%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15,"
        "%16,%17,%18,%19,%20,%21,%22,%23,%24,%25,%26,%27,%28,%29,%30,%31}, [%32];"
        : "=r"(r[0]), "=r"(r[1]), "=r"(r[2]), "=r"(r[3]), "=r"(r[4]), "=r"(r[5]), "=r"(r[6]), "=r"(r[7]),
          "=r"(r[8]), "=r"(r[9]), "=r"(r[10]), "=r"(r[11]), "=r"(r[12]), "=r"(r[13]), "=r"(r[14]), "=r"(r[15]),
          "=r"(r[16]), "=r"(r[17]), "=r"(r[18]), "=r"(r[19]), "=r"(r[20]), "=r"(r[21]), "=r"(r[22]), "=r"(r[23]),
          "=r"(r[24]), "=r"(r[25]), "=r"(r[26]), "=r"(r[27]), "=r"(r[28]), "=r"(r[29]), "=r"(r[30]), "=r"(r[31])
        : "r"(taddr));
    asm volatile("tcgen05.wait::ld.sync.aligned;" ::: "memory");
#pragma unroll
    for (int i = 0; i < 32; i++) v[i] = __uint_as_float(r[i]);
}

// byte offset of the 16-byte chunk (row, k = 4*kchunk .. 4*kchunk+3) in a K-major SW128
// tile: rows of 32 fp32 = 128 B, 8-row atoms of 1024 B, chunk index XOR (row & 7).
__device__ __forceinline__ uint32_t kmaj_off(int row, int kchunk)
{
    return (uint32_t)((row >> 3) * 1024 + (row & 7) * 128 + ((kchunk ^ (row & 7)) << 4));
}

template <int BN>
struct Cfg {
    static constexpr int STAGES = BN >= 256 ? 2 : 3;
    static constexpr int A_BYTES = BM * BK * 4;   // 16 KB
    static constexpr int B_BYTES = BN * BK * 4;
    static constexpr int STAGE = 2 * A_BYTES + 2 * B_BYTES;
    static constexpr int SMEM = STAGES * STAGE + 1024 /*align*/ + 256 /*barriers*/;
    static constexpr int APER = BM * BK / 4 / NPROD;        // A float4 per thread (4)
    static constexpr int BPER = BN * BK / 4 / NPROD;        // B float4 per thread (BN/32)
};

__device__ __forceinline__ float4 split_big(float4 v)
{
    return make_float4(to_tf32(v.x), to_tf32(v.y), to_tf32(v.z), to_tf32(v.w));
}
__device__ __forceinline__ void sts128(uint32_t addr, float4 v)
{
    asm volatile("st.shared.v4.f32 [%0], {%1,%2,%3,%4};" ::"r"(addr), "f"(v.x), "f"(v.y), "f"(v.z), "f"(v.w)
                 : "memory");
}
__device__ __forceinline__ void store_split(uint8_t *big, uint8_t *small, uint32_t off, float4 v)
{
    const float4 b = split_big(v);
    sts128(smem_u32(big) + off, b);
    sts128(smem_u32(small) + off, make_float4(v.x - b.x, v.y - b.y, v.z - b.z, v.w - b.w));
}

// NN B operand: producer thread t, unit p holds the 4 (k) x 4 (n) block at k-chunk kq,
// n-quad nq.  Lane bits: [0] = nq bit 0, [1:2] = kq bits 0-1, [3:4] = nq bits 1-2; the
// warp/unit index supplies kq bit 2 and the high nq bits.  A warp's LDG.128 then covers 4
// k-rows x 128 contiguous bytes, and the 8 lanes of each STS.128 phase (rows 8m+i, 8m+4+i;
// 4 consecutive k-chunks) land on 8 distinct swizzled chunks: conflict-free with the
// transpose done in registers at compile-time indices.
template <int BN>
__device__ __forceinline__ void nn_unit(int t, int p, int &kq, int &nq)
{
    static_assert(BN >= 128 && BN % 32 == 0, "nn_unit needs >= 1 unit per producer thread");
    constexpr int NG = BN / 32;
    const int lane = t & 31, idx = (t >> 5) + p * (NPROD / 32);
    kq = ((lane >> 1) & 3) | ((idx / NG) << 2);
    nq = (lane & 1) | (((lane >> 3) & 3) << 1) | ((idx % NG) << 3);
}

// a batch of equally shaped products, one per blockIdx.z (element strides; the inverse form of
// tc_inv.cuh), and beta0: C_in taken as zero (C is written, not read)
struct GemmBatch {
    int64_t a = 0, b = 0, c = 0;
    int beta0 = 0;
};

template <int BN, bool NT, bool NEG, bool LOWER, bool BATCH = false>
__global__ void __launch_bounds__(NTHREADS, 1)
tc_gemm_kernel(int M, int N, int K, const float *__restrict__ A, int lda, const float *__restrict__ B, int ldb,
               float *__restrict__ C, int ldc, GemmBatch bt, TaskCtx ctx)
{
    ctx_begin(ctx);
    if (BATCH) {   // a compile-time switch: the batch fields cost the tile kernel a register
        A += blockIdx.z * bt.a;
        B += blockIdx.z * bt.b;
        C += blockIdx.z * bt.c;
    }
    using G = Cfg<BN>;
    constexpr int STAGES = G::STAGES;
    extern __shared__ uint8_t smem_raw[];
    // 1024-byte aligned, indexed from the __shared__ array so accesses stay LDS/STS
    uint8_t *smem = smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u);
    uint64_t *full = (uint64_t *)(smem + STAGES * G::STAGE);
    uint64_t *empty = full + STAGES;
    uint64_t *acc_full = empty + STAGES;
    uint32_t *tmem_slot = (uint32_t *)(acc_full + 1);

    const int m0 = blockIdx.y * BM, n0 = blockIdx.x * BN;
    if (LOWER && n0 >= m0 + BM) {
        ctx_end(ctx);
        return;
    }
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int nk = K / BK;

    if (threadIdx.x == 0) {
        for (int s = 0; s < STAGES; s++) {
            mbar_init(&full[s], NPROD / 32);   // one arrive per producer warp
            mbar_init(&empty[s], 1);
        }
        mbar_init(acc_full, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    if (warp == NPROD / 32) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(tmem_slot)),
                     "r"((uint32_t)(2 * BN)));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
    }
    tc_fence_before();
    __syncthreads();
    tc_fence_after();
    const uint32_t tmem = *tmem_slot;

    if (warp < NPROD / 32) {
        // ------------------------------------------------------------ producers
        const int t = threadIdx.x;
        constexpr int APER = G::APER, BPER = G::BPER;
        const float4 z4 = make_float4(0.f, 0.f, 0.f, 0.f);
        auto load = [&](float4 (&ra)[APER], float4 (&rb)[BPER], int kb) {
            const int k0 = kb * BK;
#pragma unroll
            for (int p = 0; p < APER; p++) {
                const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                ra[p] = (m0 + row < M) ? __ldg(reinterpret_cast<const float4 *>(A + (int64_t)(m0 + row) * lda + k0 + 4 * c)) : z4;
            }
            if (NT) {
#pragma unroll
                for (int p = 0; p < BPER; p++) {
                    const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                    rb[p] = (n0 + row < N) ? __ldg(reinterpret_cast<const float4 *>(B + (int64_t)(n0 + row) * ldb + k0 + 4 * c)) : z4;
                }
            } else {
                // NN: 4 (k) x 4 (n) blocks, see nn_unit
#pragma unroll
                for (int p = 0; p < BPER / 4; p++) {
                    int kq, nq;
                    nn_unit<BN>(t, p, kq, nq);
                    const bool ok = n0 + 4 * nq < N;
#pragma unroll
                    for (int i = 0; i < 4; i++)
                        rb[4 * p + i] = ok ? __ldg(reinterpret_cast<const float4 *>(B + (int64_t)(k0 + 4 * kq + i) * ldb + n0 + 4 * nq)) : z4;
                }
            }
        };
        auto produce = [&](float4 (&ra)[APER], float4 (&rb)[BPER], int kb) {
            const int s = kb % STAGES;
            if (kb >= STAGES) mbar_wait(&empty[s], ((kb / STAGES) - 1) & 1);
            uint8_t *st = smem + s * G::STAGE;
            uint8_t *a_big = st, *a_small = st + G::A_BYTES;
            uint8_t *b_big = st + 2 * G::A_BYTES, *b_small = b_big + G::B_BYTES;
#pragma unroll
            for (int p = 0; p < APER; p++) {
                const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                store_split(a_big, a_small, kmaj_off(row, c), ra[p]);
            }
            if (NT) {
#pragma unroll
                for (int p = 0; p < BPER; p++) {
                    const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                    store_split(b_big, b_small, kmaj_off(row, c), rb[p]);
                }
            } else {
#pragma unroll
                for (int p = 0; p < BPER / 4; p++) {
                    int kq, nq;
                    nn_unit<BN>(t, p, kq, nq);
                    const float4 r0 = rb[4 * p], r1 = rb[4 * p + 1], r2 = rb[4 * p + 2], r3 = rb[4 * p + 3];
                    // column n' of the 4x4 block = K-major 16-byte chunk of row n = 4nq+n'
                    store_split(b_big, b_small, kmaj_off(4 * nq + 0, kq), make_float4(r0.x, r1.x, r2.x, r3.x));
                    store_split(b_big, b_small, kmaj_off(4 * nq + 1, kq), make_float4(r0.y, r1.y, r2.y, r3.y));
                    store_split(b_big, b_small, kmaj_off(4 * nq + 2, kq), make_float4(r0.z, r1.z, r2.z, r3.z));
                    store_split(b_big, b_small, kmaj_off(4 * nq + 3, kq), make_float4(r0.w, r1.w, r2.w, r3.w));
                }
            }
            fence_proxy_async();
            __syncwarp();                            // the warp's stores + fences precede...
            if (lane == 0) mbar_arrive(&full[s]);    // ...one release-arrive per warp
        };
        // C_in staging into TMEM columns [BN, 2BN) (this warp: lane quarter eq, column half
        // eh), one 32-column chunk after each of the first k-blocks so that the MMAs start
        // at once and the chunk loads hide behind the queued stages
        const int eq = warp & 3, eh = warp >> 2;
        const int erow = m0 + eq * 32 + lane;
        constexpr int NCH = BN / 64;
        auto stage_c = [&](int c) {
            const int col0 = eh * (BN / 2) + c * 32;
            float v[32];
            const float *crow = C + (int64_t)erow * ldc + n0 + col0;
#pragma unroll
            for (int j = 0; j < 8; j++) {
                const float4 x = (!(BATCH && bt.beta0) && erow < M && n0 + col0 + 4 * j < N) ? *reinterpret_cast<const float4 *>(crow + 4 * j) : z4;
                v[4 * j] = x.x; v[4 * j + 1] = x.y; v[4 * j + 2] = x.z; v[4 * j + 3] = x.w;
            }
            tmem_st32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)(BN + col0), v);
        };
        // D k-blocks of loads in flight (register buffers, loop unrolled by D): 2 for the wide
        // tile, 3 for BN = 128 (its small grids are latency-bound: the inverse form)
        int staged = 0;
        if constexpr (BN > 128) {
            float4 ra0[APER], rb0[BPER], ra1[APER], rb1[BPER];
            load(ra0, rb0, 0);
            if (nk > 1) load(ra1, rb1, 1);
            for (int kb = 0; kb < nk; kb += 2) {
                produce(ra0, rb0, kb);
                if (kb + 2 < nk) load(ra0, rb0, kb + 2);
                if (staged < NCH) stage_c(staged++);
                if (kb + 1 < nk) {
                    produce(ra1, rb1, kb + 1);
                    if (kb + 3 < nk) load(ra1, rb1, kb + 3);
                    if (staged < NCH) stage_c(staged++);
                }
            }
        } else {
            constexpr int D = 3;
            float4 ra[D][APER], rb[D][BPER];
#pragma unroll
            for (int d = 0; d < D; d++)
                if (d < nk) load(ra[d], rb[d], d);
            for (int kb = 0; kb < nk; kb += D) {
#pragma unroll
                for (int d = 0; d < D; d++) {
                    if (kb + d < nk) {
                        produce(ra[d], rb[d], kb + d);
                        if (kb + d + D < nk) load(ra[d], rb[d], kb + d + D);
                        if (staged < NCH) stage_c(staged++);
                    }
                }
            }
        }
        while (staged < NCH) stage_c(staged++);
        asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");

        // ------------------------------------------------------------ epilogue
        mbar_wait(acc_full, 0);
        tc_fence_after();
        // C_in was staged in TMEM columns [BN, 2BN): C = C_in + acc in fp32 round-to-nearest
        // (the accumulation onto C is NOT done by the MMA: the tensor core's fp32
        // accumulate is not round-to-nearest and loses precision on a large addend).
#pragma unroll 1
        for (int c = 0; c < BN / 64; c++) {
            const int col0 = eh * (BN / 2) + c * 32;
            float v[32], cv[32];
            tmem_ld32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)col0, v);
            tmem_ld32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)(BN + col0), cv);
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
    } else {
        // ------------------------------------------------------------ MMA issuer
        constexpr uint32_t idesc = make_idesc(BM, BN, NEG, false);
        for (int kb = 0; kb < nk; kb++) {
            const int s = kb % STAGES;
            mbar_wait(&full[s], (kb / STAGES) & 1);
            tc_fence_after();
            if (lane == 0) {
                uint8_t *st = smem + s * G::STAGE;
                const uint32_t a_big = smem_u32(st), a_small = a_big + G::A_BYTES;
                const uint32_t b_big = a_big + 2 * G::A_BYTES, b_small = b_big + G::B_BYTES;
#pragma unroll
                for (int kk = 0; kk < BK / 8; kk++) {
                    // K-major SW128: the k-step advances 32 B inside the 128 B swizzled row
                    const uint32_t o = kk * 32;
                    const uint64_t dAb = make_desc(a_big + o, 16, 1024), dAs = make_desc(a_small + o, 16, 1024);
                    const uint64_t dBb = make_desc(b_big + o, 16, 1024), dBs = make_desc(b_small + o, 16, 1024);
                    const uint32_t first = (kb == 0 && kk == 0) ? 0u : 1u;
                    mma_tf32(tmem, dAb, dBb, idesc, first);
                    mma_tf32(tmem, dAb, dBs, idesc, 1u);
                    mma_tf32(tmem, dAs, dBb, idesc, 1u);
                }
                mma_commit(&empty[s]);
                if (kb == nk - 1) mma_commit(acc_full);
            }
            __syncwarp();
        }
    }

    tc_fence_before();
    __syncthreads();
    if (warp == NPROD / 32) {
        tc_fence_after();
        asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"((uint32_t)(2 * BN)));
    }
    ctx_end(ctx);
}

// Host launcher: K multiple of 32; lda/ldb/ldc multiples of 4 and 16-byte aligned bases.
// BATCH: count products along blockIdx.z with the element strides of bt (bt.beta0: C_in = 0)
template <bool NT, bool NEG, bool LOWER, int BN = 256, bool BATCH = false>
inline int tc_gemm(int M, int N, int K, const float *A, int lda, const float *B, int ldb, float *C, int ldc,
                   cudaStream_t s, const TaskCtx &ctx = TaskCtx(), const GemmBatch &bt = GemmBatch(), int count = 1)
{
    if (M <= 0 || N <= 0) return 0;
    if (K % BK || (!BATCH && (count != 1 || bt.beta0))) return -1;
    auto kern = tc_gemm_kernel<BN, NT, NEG, LOWER, BATCH>;
    constexpr int smem = Cfg<BN>::SMEM;
    static bool attr[64] = {};
    int dev = 0;
    cudaGetDevice(&dev);
    if (!attr[dev & 63]) {
        cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
        attr[dev & 63] = true;
    }
    dim3 grid((N + BN - 1) / BN, (M + BM - 1) / BM, count);
    // The tensor core's fp32 accumulation does not round to nearest: its error grows linearly
    // with the accumulated K (measured relF of a b x b MATMUL: 7.2e-6 at K = 1024, 1.4e-5 at 2048,
    // 2.9e-5 at 4096).  K is therefore cut into chunks of at most kKChunk, one launch each; every
    // launch adds its chunk to C in fp32 round-to-nearest (the C_in path), which keeps every K at
    // the K = 1024 error (fp32-class gate, BASELINE north star)
    const TaskCtx c = ctx_for(ctx, kern, NTHREADS, smem);
    for (int k0 = 0; k0 < K; k0 += kKChunk) {
        const int kc = K - k0 < kKChunk ? K - k0 : kKChunk;
        GemmBatch bc = bt;
        if (k0 > 0) bc.beta0 = 0;   // later chunks accumulate onto the first one's result
        count_launch();
        kern<<<grid, NTHREADS, smem, s>>>(M, N, kc, A + k0, lda, B + (NT ? (int64_t)k0 : (int64_t)k0 * ldb), ldb, C, ldc,
                                          bc, c);
    }
    return 0;
}

}  // namespace tc
}  // namespace vsk
