// tc_trsm.cuh — single-launch tcgen05 3xTF32 triangular solve (trsm task, tc_3xtf32 version,
// also the panel solve inside potrf).
//
//   X L^T = B  (right side, L lower, transposed, non-unit; reading R5), X overwrites B.
//   rows x n block X (ldx), n x n lower L (ldl); n a multiple of P = 64.
//
// Left-looking over column panels J of width P, each CTA owning 128 rows (rows are
// independent):
//   1. T_J = B[:, J] - X[:, <J] L[J, <J]^T : tcgen05 3xTF32 MMA (M=128, N=P, K=J*P),
//      A = the CTA's own already-solved X columns (re-read from global/L2 with coherent
//      loads), B = L rows of panel J (K-major), accumulator in TMEM (P columns);
//   2. X[:, J] = T_J L_JJ^{-T}: each of 128 threads owns one row, tcgen05.ld its P
//      accumulator values and runs the column-oriented forward substitution
//      x_c = t_c / L_cc; t_j -= x_c L_jc (j > c) against L_JJ staged in shared memory
//      (IEEE division, so integer problems stay exact), then stores the row segment.
// One launch replaces the 2 * n/P launches of the blocked version.
#pragma once
#include "tc_gemm.cuh"

namespace vsk {
namespace tc {

constexpr int TRSM_P = 64;

struct TrsmCfg {
    static constexpr int STAGES = 3;
    static constexpr int A_BYTES = BM * BK * 4;        // 16 KB
    static constexpr int B_BYTES = TRSM_P * BK * 4;    // 8 KB
    static constexpr int STAGE = 2 * A_BYTES + 2 * B_BYTES;
    static constexpr int LS_BYTES = TRSM_P * (TRSM_P + 1) * 4;
    static constexpr int SMEM = STAGES * STAGE + LS_BYTES + 1024 + 256;
    static constexpr int APER = BM * BK / 4 / NPROD;      // 4
    static constexpr int BPER = TRSM_P * BK / 4 / NPROD;  // 2
};

__device__ __forceinline__ float rcp_approx(float x)
{
    float r;
    asm("rcp.approx.ftz.f32 %0, %1;" : "=f"(r) : "f"(x));
    return r;
}
// t / l without the IEEE-division slow-path call (which forces the per-thread row into
// local memory): x0 = t r, one Newton correction x = x0 + (t - x0 l) r.  For a positive
// normal l this is the correctly rounded quotient whenever t / l is representable
// (integer problems stay exact) and within 1 ulp otherwise.
__device__ __forceinline__ float div_nr(float t, float l, float r)
{
    const float x0 = t * r;
    return fmaf(fmaf(-x0, l, t), r, x0);
}

__device__ __forceinline__ float4 ld_f4_coherent(const float *p)
{
    float4 v;
    asm volatile("ld.global.v4.f32 {%0,%1,%2,%3}, [%4];" : "=f"(v.x), "=f"(v.y), "=f"(v.z), "=f"(v.w) : "l"(p));
    return v;
}

__global__ void __launch_bounds__(NTHREADS, 1)
tc_trsm_kernel(int rows, int n, const float *__restrict__ L, int ldl, float *X, int ldx, TaskCtx ctx)
{
    ctx_begin(ctx);
    using G = TrsmCfg;
    constexpr int P = TRSM_P, STAGES = G::STAGES;
    extern __shared__ uint8_t smem_raw[];
    uint8_t *smem = (uint8_t *)(((uintptr_t)smem_raw + 1023) & ~(uintptr_t)1023);
    float(*Ls)[P + 1] = reinterpret_cast<float(*)[P + 1]>(smem + STAGES * G::STAGE);
    __shared__ float Lr[P];   // approximate reciprocals of the diagonal of L_JJ
    uint64_t *full = (uint64_t *)(smem + STAGES * G::STAGE + G::LS_BYTES);
    uint64_t *empty = full + STAGES;
    uint64_t *acc_full = empty + STAGES;
    uint32_t *tmem_slot = (uint32_t *)(acc_full + 1);

    const int m0 = blockIdx.x * BM;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    if (threadIdx.x == 0) {
        for (int s = 0; s < STAGES; s++) {
            mbar_init(&full[s], NPROD / 32);
            mbar_init(&empty[s], 1);
        }
        mbar_init(acc_full, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    if (warp == NPROD / 32) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(tmem_slot)),
                     "r"((uint32_t)P));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
    }
    tc_fence_before();
    __syncthreads();
    tc_fence_after();
    const uint32_t tmem = *tmem_slot;
    const int npanels = n / P;
    int gkb = 0;        // global k-block counter (barrier phases run across panels)
    int acc_uses = 0;   // completed acc_full phases

    for (int J = 0; J < npanels; J++) {
        const int c0 = J * P;
        const int nk = c0 / BK;
        if (warp < NPROD / 32) {
            const int t = threadIdx.x;
            // stage L_JJ (lower) for the solve
            {
                constexpr int PER = P * P / NPROD;   // batched loads, then stores
                float tmp[PER];
#pragma unroll
                for (int q = 0; q < PER; q++) {
                    const int e = t + q * NPROD, i = e / P, j = e % P;
                    tmp[q] = j <= i ? __ldg(L + (int64_t)(c0 + i) * ldl + c0 + j) : 0.f;
                }
#pragma unroll
                for (int q = 0; q < PER; q++) {
                    const int e = t + q * NPROD, i = e / P, j = e % P;
                    Ls[i][j] = tmp[q];
                }
                if (t < P) Lr[t] = rcp_approx(__ldg(L + (int64_t)(c0 + t) * ldl + c0 + t));
            }
            // ---- producers: A = X[m0.., 0:c0] (coherent loads), B = L[c0..c0+P, 0:c0] (K-major)
            constexpr int APER = G::APER, BPER = G::BPER;
            const float4 z4 = make_float4(0.f, 0.f, 0.f, 0.f);
            auto load = [&](float4 (&ra)[APER], float4 (&rb)[BPER], int kb) {
                const int k0 = kb * BK;
#pragma unroll
                for (int p = 0; p < APER; p++) {
                    const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                    ra[p] = (m0 + row < rows) ? ld_f4_coherent(X + (int64_t)(m0 + row) * ldx + k0 + 4 * c) : z4;
                }
#pragma unroll
                for (int p = 0; p < BPER; p++) {
                    const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                    rb[p] = __ldg(reinterpret_cast<const float4 *>(L + (int64_t)(c0 + row) * ldl + k0 + 4 * c));
                }
            };
            auto produce = [&](float4 (&ra)[APER], float4 (&rb)[BPER]) {
                const int s = gkb % STAGES;
                if (gkb >= STAGES) mbar_wait(&empty[s], ((gkb / STAGES) - 1) & 1);
                uint8_t *st = smem + s * G::STAGE;
                uint8_t *a_big = st, *a_small = st + G::A_BYTES;
                uint8_t *b_big = st + 2 * G::A_BYTES, *b_small = b_big + G::B_BYTES;
#pragma unroll
                for (int p = 0; p < APER; p++) {
                    const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                    store_split(a_big, a_small, kmaj_off(row, c), ra[p]);
                }
#pragma unroll
                for (int p = 0; p < BPER; p++) {
                    const int f = t + p * NPROD, row = f >> 3, c = f & 7;
                    store_split(b_big, b_small, kmaj_off(row, c), rb[p]);
                }
                fence_proxy_async();
                __syncwarp();
                if (lane == 0) mbar_arrive(&full[s]);   // one release-arrive per producer warp
                gkb++;
            };
            if (nk > 0) {
                float4 ra0[APER], rb0[BPER], ra1[APER], rb1[BPER];
                load(ra0, rb0, 0);
                if (nk > 1) load(ra1, rb1, 1);
                for (int kb = 0; kb < nk; kb += 2) {
                    produce(ra0, rb0);
                    if (kb + 2 < nk) load(ra0, rb0, kb + 2);
                    if (kb + 1 < nk) {
                        produce(ra1, rb1);
                        if (kb + 3 < nk) load(ra1, rb1, kb + 3);
                    }
                }
            }
            asm volatile("bar.sync 1, %0;" ::"r"(NPROD));     // Ls staged by all producers
            // ---- solve: warps 0-3, one row per thread
            if (warp < 4) {
                const int row = m0 + warp * 32 + lane;
                float tv[P];
                if (nk > 0) {
                    mbar_wait(acc_full, acc_uses & 1);
                    tc_fence_after();
                    float v[32];
#pragma unroll
                    for (int h = 0; h < P / 32; h++) {
                        tmem_ld32(tmem + ((uint32_t)(warp * 32) << 16) + (uint32_t)(h * 32), v);
#pragma unroll
                        for (int i = 0; i < 32; i++) tv[h * 32 + i] = -v[i];
                    }
                } else {
#pragma unroll
                    for (int i = 0; i < P; i++) tv[i] = 0.f;
                }
                if (row < rows) {
                    float *xr = X + (int64_t)row * ldx + c0;
#pragma unroll
                    for (int q = 0; q < P / 4; q++) {
                        const float4 bq = ld_f4_coherent(xr + 4 * q);
                        tv[4 * q + 0] += bq.x; tv[4 * q + 1] += bq.y; tv[4 * q + 2] += bq.z; tv[4 * q + 3] += bq.w;
                    }
#pragma unroll
                    for (int c = 0; c < P; c++) {
                        tv[c] = div_nr(tv[c], Ls[c][c], Lr[c]);
#pragma unroll
                        for (int j = 0; j < P; j++)
                            if (j > c) tv[j] = fmaf(-tv[c], Ls[j][c], tv[j]);
                    }
#pragma unroll
                    for (int q = 0; q < P / 4; q++)
                        *reinterpret_cast<float4 *>(xr + 4 * q) = make_float4(tv[4 * q], tv[4 * q + 1], tv[4 * q + 2], tv[4 * q + 3]);
                }
            }
        } else {
            // ---- MMA issuer
            constexpr uint32_t idesc = make_idesc(BM, P, false, false);
            int kb_local = 0;
            for (int kb = 0; kb < nk; kb++, kb_local++) {
                const int g = gkb + kb;
                const int s = g % STAGES;
                mbar_wait(&full[s], (g / STAGES) & 1);
                tc_fence_after();
                if (lane == 0) {
                    uint8_t *st = smem + s * G::STAGE;
                    const uint32_t a_big = smem_u32(st), a_small = a_big + G::A_BYTES;
                    const uint32_t b_big = a_big + 2 * G::A_BYTES, b_small = b_big + G::B_BYTES;
#pragma unroll
                    for (int kk = 0; kk < BK / 8; kk++) {
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
            gkb += nk;
        }
        if (nk > 0) acc_uses++;
        // panel boundary: X[:, J] visible to the next panel's producers, TMEM / Ls reusable
        tc_fence_before();
        __threadfence_block();
        __syncthreads();
        tc_fence_after();
    }

    if (warp == NPROD / 32) {
        asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"((uint32_t)P));
    }
    ctx_end(ctx);
}

inline int tc_trsm(int rows, int n, const float *L, int ldl, float *X, int ldx, cudaStream_t s,
                   const TaskCtx &ctx = TaskCtx())
{
    if (rows <= 0 || n <= 0) return 0;
    if (n % TRSM_P) return -1;
    constexpr int smem = TrsmCfg::SMEM;
    static bool attr[64] = {};
    int dev = 0;
    cudaGetDevice(&dev);
    if (!attr[dev & 63]) {
        cudaFuncSetAttribute(tc_trsm_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
        attr[dev & 63] = true;
    }
    count_launch();
    tc_trsm_kernel<<<(rows + BM - 1) / BM, NTHREADS, smem, s>>>(rows, n, L, ldl, X, ldx, ctx);
    return 0;
}

}  // namespace tc
}  // namespace vsk
