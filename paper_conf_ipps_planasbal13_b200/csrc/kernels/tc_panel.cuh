// tc_panel.cuh — single-launch tcgen05 3xTF32 left-looking panel kernel: the trsm task and
// the potrf task of the tc_3xtf32 version (reading R5; PAPER.md L697-699 for the
// algorithm of Cholesky, R9 for info).
//
//   TRSM:  X L^T = B (right side, L lower, transposed, non-unit), X overwrites B;
//          rows x n block X (ldx), n x n lower L (ldl).
//   POTRF: A = L L^T in place (n x n, lower triangle read and written, the strict upper
//          triangle untouched, R7); first non-positive pivot -> *info = k_base + col + 1.
// n a multiple of 64.  Each CTA owns 128 rows (TMEM lanes = rows) and walks the column
// panels J (P = 128 wide, the last one possibly 64) left to right:
//   1. T_J = B[:, J] - X[:, <J] L[J, <J]^T     (POTRF: A[:, J] - L[:, <J] L[J, <J]^T)
//      tcgen05 3xTF32 MMA, M = 128, N = 128, K = 128 J, into one of two TMEM
//      accumulators (panel parity) so that the MMA of panel J+1 runs while panel J is
//      being solved.  A operand = the CTA's own solved columns, B operand = the panel's
//      L rows; the k-blocks that need the columns solved in panel J wait for that panel
//      only (mbarrier xdone; a per-k-block variant measured slower: 527 vs 490 us).
//   2. epilogue warps, one row each, per 16-column sub-block sb (compact code: a 16 x 16
//      step is the only unrolled unit):
//        x = b - acc[sb]  (b = the tile's current values, staged in TMEM by the producers);
//        TRSM / POTRF below the diagonal: forward substitution against L_JJ staged
//          (transposed) in shared memory (x_c = t_c / l_cc; t_j -= x_c l_jc);
//        POTRF diagonal CTA (CTA J holds panel J's diagonal block): per 16-column
//          sub-block, the warp holding its 16 diagonal rows factors them with shuffles
//          (l_cc = sqrt(t_c), x = t / l, t_j -= x l_jc), publishes L_sb, and the rows below
//          solve against it (two named barriers per sub-block; round 1: two per column);
//        store x; acc[t] += x L[t, sb]^T for the later sub-blocks t (tcgen05.ld/st).
// Roles: warps 0-3 producers (LDG -> split big/small -> 128B-swizzled K-major smem); warp 0
// also allocates TMEM and, once all four producer warps filled a stage, issues its MMAs;
// warps 4-7 epilogue (TMEM lane quarter = warp % 4).
// POTRF: the other CTAs wait, through a per-launch progress word per CTA (release /
// acquire at gpu scope), for CTA J to have finished panels < J before loading panel J's
// L rows as MMA operand, and panel J before staging L_JJ.  Every CTA only waits on
// lower-numbered CTAs of the same grid, which never wait on it: each one eventually
// becomes resident and the launch cannot deadlock.
// Division: rcp.approx + one Newton step (correctly rounded when the quotient is
// representable: integer problems stay exact); sqrt is IEEE.
#pragma once
#include <atomic>
#include <cstdio>
#include <cstdlib>

#include "tc_gemm.cuh"

namespace vsk {
namespace tc {

// Optional per-CTA, per-panel timeline (a probe builds with -DVS_PANEL_TRACE):
// [cta][panel][0] epilogue: flag seen, [1] L_JJ staged, [2] accumulator ready, [3] panel solved,
// [4] producer: flag seen (potrf), [5] producer: last k-block issued, [6 + 2 sb] sub-block sb
// solved (before the cross update), [7 + 2 sb] its cross update done
#ifdef VS_PANEL_TRACE
__device__ unsigned long long g_panel_trace[32][32][24];
__device__ long long g_panel_clk[32][32][24];   // SM clock64 at the same points
__device__ unsigned long long g_panel_trace_id;  // 0: every launch, else that potrf launch id only
#define PANEL_T(J, i)                                                                  \
    do {                                                                               \
        if (g_panel_trace_id == 0 || g_panel_trace_id == launch_id) {                  \
            unsigned long long t_;                                                     \
            asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t_));                     \
            g_panel_trace[blockIdx.x & 31][(J) & 31][i] = t_;                          \
            g_panel_clk[blockIdx.x & 31][(J) & 31][i] = clock64();                     \
        }                                                                              \
    } while (0)
#else
#define PANEL_T(J, i)
#endif

constexpr int PNL = 128;   // panel width (= BM: panel J's diagonal block is CTA J's rows)
constexpr int PSB = 16;    // solve sub-block
constexpr int kFlagSlots = 4096;
constexpr int kFlagCtas = 32;   // n <= 4096 -> at most 32 CTAs per potrf launch
constexpr int PTHREADS = 256;   // 4 producer warps (warp 0 also issues the MMAs) + 4 epilogue
                                // warps: 8 warps keep the 255-register budget (9 would cap at 168)

struct PanelCfg {
    static constexpr int STAGES = 2;
    static constexpr int NP = 128;                          // producer threads
    static constexpr int A_BYTES = BM * BK * 4;             // 16 KB
    static constexpr int B_BYTES = PNL * BK * 4;            // 16 KB
    static constexpr int STAGE = 2 * A_BYTES + 2 * B_BYTES; // 64 KB
    static constexpr int LD = PNL + 4;                      // Lt row stride (16-byte rows)
    static constexpr int LT_BYTES = PNL * LD * 4;           // 66 KB
    static constexpr int XS_A = BM * 64;                    // 8 KB: 128 rows x 16 fp32 (SW64), one part
    static constexpr int XS_B = (PNL - 16) * 64;            // 7 KB: at most 112 rows of L_JJ, one part
    static constexpr int XS_BYTES = 2 * XS_A + 2 * XS_B;    // cross-sub-block update operands
    static constexpr int SMEM = STAGES * STAGE + LT_BYTES + XS_BYTES + 1024 + 256;
    static constexpr int APER = BM * BK / 4 / NP;           // 8
    static constexpr int BPER = PNL * BK / 4 / NP;          // 8
};

// progress words of the potrf launches: slot = launch id % kFlagSlots, value =
// (launch id << 8) | panels completed; ids grow, so no reset is needed between launches
__device__ unsigned long long g_panel_flags[kFlagSlots][kFlagCtas];

__device__ __forceinline__ float rcp_approx(float x)
{
    float r;
    asm("rcp.approx.ftz.f32 %0, %1;" : "=f"(r) : "f"(x));
    return r;
}
// t / l: x0 = t r, one Newton correction x = x0 + (t - x0 l) r
__device__ __forceinline__ float div_nr(float t, float l, float r)
{
    const float x0 = t * r;
    return fmaf(fmaf(-x0, l, t), r, x0);
}
// L2-coherent loads (data written by this or other CTAs during the launch)
__device__ __forceinline__ float4 ld_f4_cg(const float *p)
{
    float4 v;
    asm volatile("ld.global.cg.v4.f32 {%0,%1,%2,%3}, [%4];" : "=f"(v.x), "=f"(v.y), "=f"(v.z), "=f"(v.w) : "l"(p));
    return v;
}
__device__ __forceinline__ float ld_f_cg(const float *p)
{
    float v;
    asm volatile("ld.global.cg.f32 %0, [%1];" : "=f"(v) : "l"(p));
    return v;
}
__device__ __forceinline__ unsigned long long ld_acquire(const unsigned long long *p)
{
    unsigned long long v;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ void st_release(unsigned long long *p, unsigned long long v)
{
    asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ void wait_flag(const unsigned long long *p, unsigned long long need)
{
    while (ld_acquire(p) < need) __nanosleep(64);
}

__device__ __forceinline__ void tmem_ld16(uint32_t taddr, float (&v)[16])
{
    uint32_t r[16];
    asm volatile(
        "tcgen05.ld.sync.aligned.32x32b.x16.b32 {%0,%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15}, [%16];"
        : "=r"(r[0]), "=r"(r[1]), "=r"(r[2]), "=r"(r[3]), "=r"(r[4]), "=r"(r[5]), "=r"(r[6]), "=r"(r[7]),
          "=r"(r[8]), "=r"(r[9]), "=r"(r[10]), "=r"(r[11]), "=r"(r[12]), "=r"(r[13]), "=r"(r[14]), "=r"(r[15])
        : "r"(taddr));
    asm volatile("tcgen05.wait::ld.sync.aligned;" ::: "memory");
#pragma unroll
    for (int i = 0; i < 16; i++) v[i] = __uint_as_float(r[i]);
}
__device__ __forceinline__ void tmem_st16(uint32_t taddr, const float (&v)[16])
{
    asm volatile(
        "tcgen05.st.sync.aligned.32x32b.x16.b32 [%0], {%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15,%16};" ::"r"(
            taddr),
        "f"(v[0]), "f"(v[1]), "f"(v[2]), "f"(v[3]), "f"(v[4]), "f"(v[5]), "f"(v[6]), "f"(v[7]), "f"(v[8]), "f"(v[9]),
        "f"(v[10]), "f"(v[11]), "f"(v[12]), "f"(v[13]), "f"(v[14]), "f"(v[15])
        : "memory");
    asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");
}
// split-phase TMEM access for software pipelining: the wait takes the destination
// registers as in/out operands so that no use of them is scheduled before it
__device__ __forceinline__ void tmem_ld16_issue(uint32_t taddr, float (&v)[16])
{
    asm volatile(
        "tcgen05.ld.sync.aligned.32x32b.x16.b32 {%0,%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15}, [%16];"
        : "=f"(v[0]), "=f"(v[1]), "=f"(v[2]), "=f"(v[3]), "=f"(v[4]), "=f"(v[5]), "=f"(v[6]), "=f"(v[7]),
          "=f"(v[8]), "=f"(v[9]), "=f"(v[10]), "=f"(v[11]), "=f"(v[12]), "=f"(v[13]), "=f"(v[14]), "=f"(v[15])
        : "r"(taddr));
}
__device__ __forceinline__ void tmem_wait_ld(float (&v)[16])
{
    asm volatile("tcgen05.wait::ld.sync.aligned;"
                 : "+f"(v[0]), "+f"(v[1]), "+f"(v[2]), "+f"(v[3]), "+f"(v[4]), "+f"(v[5]), "+f"(v[6]), "+f"(v[7]),
                   "+f"(v[8]), "+f"(v[9]), "+f"(v[10]), "+f"(v[11]), "+f"(v[12]), "+f"(v[13]), "+f"(v[14]), "+f"(v[15])
                 :
                 : "memory");
}
__device__ __forceinline__ void tmem_st16_issue(uint32_t taddr, const float (&v)[16])
{
    asm volatile(
        "tcgen05.st.sync.aligned.32x32b.x16.b32 [%0], {%1,%2,%3,%4,%5,%6,%7,%8,%9,%10,%11,%12,%13,%14,%15,%16};" ::"r"(
            taddr),
        "f"(v[0]), "f"(v[1]), "f"(v[2]), "f"(v[3]), "f"(v[4]), "f"(v[5]), "f"(v[6]), "f"(v[7]), "f"(v[8]), "f"(v[9]),
        "f"(v[10]), "f"(v[11]), "f"(v[12]), "f"(v[13]), "f"(v[14]), "f"(v[15])
        : "memory");
}
__device__ __forceinline__ void tmem_wait_st() { asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory"); }
// POTRF operand images (tc_potrf): per row block and 32-wide k-block the split big / small
// values in two SW64 halves (16 k each, the layout of the cross-sub-block update operands),
// bulk-stored from shared memory by the epilogue, bulk-copied into a stage by the producers
constexpr int kImgHalf = BM * 64;          // 8 KB: 128 rows x 16 fp32
constexpr int kImgKb = 4 * kImgHalf;       // 32 KB: big (2 halves) + small (2 halves)
__device__ __forceinline__ void img_expect_tx(uint64_t *bar, uint32_t bytes)
{
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes) : "memory");
}
__device__ __forceinline__ void img_g2s(uint32_t dst, const void *src, uint32_t bytes, uint64_t *bar)
{
    asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(dst),
                 "l"(src), "r"(bytes), "r"(smem_u32(bar))
                 : "memory");
}
__device__ __forceinline__ void img_s2g(void *dst, uint32_t src, uint32_t bytes)
{
    asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;" ::"l"(dst), "r"(src), "r"(bytes) : "memory");
}
__device__ __forceinline__ void img_commit() { asm volatile("cp.async.bulk.commit_group;" ::: "memory"); }
__device__ __forceinline__ void img_wait_read() { asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory"); }
__device__ __forceinline__ void img_wait_all() { asm volatile("cp.async.bulk.wait_group 0;" ::: "memory"); }
__device__ __forceinline__ void fence_proxy_async_global() { asm volatile("fence.proxy.async.global;" ::: "memory"); }
__device__ __forceinline__ void bar_epi() { asm volatile("bar.sync 2, 128;" ::: "memory"); }
// UMMA shared-memory descriptor, K-major SWIZZLE_64B (layout 4): 64-byte rows, 8-row atoms of
// 512 B (SBO), version 1 — the cross-sub-block update operands (16 fp32 of K per row)
__device__ __forceinline__ uint64_t desc_sw64(uint32_t saddr)
{
    uint64_t d = 0;
    d |= (uint64_t)((saddr & 0x3FFFF) >> 4);
    d |= (uint64_t)(16 >> 4) << 16;
    d |= (uint64_t)(512 >> 4) << 32;
    d |= (uint64_t)1 << 46;
    d |= (uint64_t)4 << 61;
    return d;
}

template <bool POTRF>
__global__ void __launch_bounds__(PTHREADS, 1)
tc_panel_kernel(int rows, int n, const float *L, int ldl, float *X, int ldx, int k_base, int *info,
                unsigned long long launch_id, int overlap, int64_t lbs, int64_t xbs, TaskCtx ctx, uint8_t *img)
{
    ctx_begin(ctx);
    L += blockIdx.y * lbs;   // TRSM batch (tc_trsm_batched): independent problems along y
    X += blockIdx.y * xbs;
    using G = PanelCfg;
    constexpr int P = PNL, STAGES = G::STAGES, LD = G::LD, NP = G::NP;
    extern __shared__ uint8_t smem_raw[];
    // 1024-byte aligned, indexed from the __shared__ array so accesses stay LDS/STS
    uint8_t *smem = smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u);
    float *Lt = reinterpret_cast<float *>(smem + STAGES * G::STAGE);   // Lt[c * LD + j] = L_JJ[j][c]
    __shared__ float Lr[P];       // reciprocals of the diagonal of L_JJ
    // XS: operands of the cross-sub-block update MMAs (1024-aligned: STAGE and LT_BYTES keep it)
    uint8_t *xs_ab = (uint8_t *)Lt + G::LT_BYTES, *xs_as = xs_ab + G::XS_A;
    uint8_t *xs_bb = xs_as + G::XS_A, *xs_bs = xs_bb + G::XS_B;
    uint64_t *full = (uint64_t *)(xs_bs + G::XS_B);
    uint64_t *empty = full + STAGES;
    uint64_t *accf = empty + STAGES;   // [2]: accumulator of panel parity b complete
    uint64_t *xdone = accf + 2;        // one phase per panel: its columns solved and stored
    uint64_t *xacc = xdone + 1;        // cross-sub-block update MMAs complete (one phase per use)
    uint64_t *bfull = xacc + 1;        // [2]: b values of panel parity b staged in TMEM (producers)
    uint64_t *pstart = bfull + 2;      // POTRF feed: the producers issued the factor panel's first MMAs
    uint32_t *tmem_slot = (uint32_t *)(pstart + 1);

    const int m0 = blockIdx.x * BM;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
#ifdef VS_PANEL_TRACE
    if (threadIdx.x == 0) {
        unsigned smid;
        asm volatile("mov.u32 %0, %%smid;" : "=r"(smid));
        g_panel_trace[blockIdx.x & 31][31][23] = smid;
    }
#endif
    unsigned long long *flags = POTRF ? g_panel_flags[launch_id % kFlagSlots] : nullptr;
    const unsigned long long tag = launch_id << 8;
    if (threadIdx.x == 0) {
        for (int s = 0; s < STAGES; s++) {
            mbar_init(&full[s], img ? 1 : NP / 32);   // images: one expect_tx arrival + the bytes
            mbar_init(&empty[s], 1);
        }
        mbar_init(&accf[0], 1);
        mbar_init(&accf[1], 1);
        mbar_init(xdone, 4);
        mbar_init(xacc, 2);   // per use: the MMA commit (or a plain arrival) + the image store's read
        mbar_init(&bfull[0], 4);
        mbar_init(&bfull[1], 4);
        mbar_init(pstart, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    if (warp == 0) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(tmem_slot)),
                     "r"((uint32_t)(4 * P)));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
    }
    tc_fence_before();
    __syncthreads();
    tc_fence_after();
    const uint32_t tmem = *tmem_slot;
    // panels this CTA takes part in: POTRF stops at the panel holding its rows' diagonal
    int npanels = (n + P - 1) / P;
    if (POTRF) npanels = min(npanels, (int)blockIdx.x + 1);
    // POTRF feed (option bit 2): the factor panel's update by the previous panel,
    // A_cc -= L_c,c-1 L_c,c-1^T, uses this CTA's own rows for both operands, so the epilogue
    // issues it sub-block by sub-block while it solves panel c-1 (operands already staged for
    // the cross-sub-block update) instead of the producers reloading the solved columns from
    // global memory after the whole panel is stored: the accumulator of the factor panel is
    // ready as soon as the solve ends (critical chain of the factorisation)
    const int fpanel = (int)blockIdx.x;
    const bool feed = POTRF && (overlap & 4) && (overlap & 1) && fpanel >= 1 && fpanel < npanels + 0 &&
                      fpanel * P < n;
    const bool feed_pk = feed && fpanel * P / BK - P / BK > 0;   // the producers issue MMAs of the factor panel

    if (warp < 4) {
        // =================================================== producers
        const int t = threadIdx.x;
        constexpr int APER = G::APER, BPER = G::BPER;
        const float4 z4 = make_float4(0.f, 0.f, 0.f, 0.f);
        int gkb = 0;
        // b values of panel J for this thread's row (the tile's current values of the panel's
        // columns: only this CTA ever writes them, when it solves panel J) -> TMEM columns
        // [2P + (J & 1) P, +ncols), lane = row: issued while the early k-blocks of panel J are
        // produced, so the epilogue's x = b - acc reads no global memory on the critical path
        // (under the GEMM flood the first sub-block's load took 10-15 us)
        const int brow = m0 + t;
        const bool browok = brow < rows;
        auto stage_b = [&](int J) {
            const int c0 = J * P, ncols = min(P, n - c0);
            const uint32_t tb = tmem + ((uint32_t)(warp * 32) << 16) + (uint32_t)(2 * P + (J & 1) * P);
            const float *src = X + (int64_t)(browok ? brow : 0) * ldx + c0;
            if (browok)   // the row's lines in flight at once; the chunks below then hit L2
                for (int q0 = 0; q0 < ncols; q0 += 32) asm volatile("prefetch.global.L2 [%0];" ::"l"(src + q0));
#pragma unroll 1
            for (int q0 = 0; q0 < ncols; q0 += 16) {   // 16 columns at a time: the k-block
                float v[16];                            // buffers ra/rb stay live in registers
#pragma unroll
                for (int i = 0; i < 4; i++) {
                    const float4 f = browok ? ld_f4_cg(src + q0 + 4 * i) : z4;
                    v[4 * i] = f.x; v[4 * i + 1] = f.y; v[4 * i + 2] = f.z; v[4 * i + 3] = f.w;
                }
                tmem_st16(tb + q0, v);
            }
            tc_fence_before();
            __syncwarp();
            if (lane == 0) mbar_arrive(&bfull[J & 1]);
        };
        for (int J = 0; J < npanels; J++) {
            const int c0 = J * P;
            // feed: the factor panel's k-blocks of panel J-1 are issued by the epilogue instead
            const int nk = (feed && J == fpanel) ? c0 / BK - P / BK : c0 / BK;
            if (nk == 0) {
                stage_b(J);
                if (feed && J == fpanel && threadIdx.x == 0) mma_commit(&accf[J & 1]);   // nothing of the producers' to wait for
                continue;
            }
            if (POTRF && J != (int)blockIdx.x) {
                // panel J's L rows (CTA J's) are final once it completed panels < J
                if (t == 0) wait_flag(&flags[J], tag | (unsigned long long)J);
                asm volatile("bar.sync 1, 128;" ::: "memory");
            }
            if (t == 0) PANEL_T(J, 4);
            // first k-block holding panel J-1's columns (overlap = 0: the whole panel waits); with
            // the feed the factor panel has none of them
            const int kb_new = (feed && J == fpanel) ? nk : (overlap & 1) ? nk - P / BK : 0;
            constexpr uint32_t idesc = make_idesc(BM, P, false, false);
            const uint32_t dt = tmem + (uint32_t)((J & 1) * P);
            int kbp = 0;   // k-block of this panel being produced
            bool waited = false;
            auto ensure = [&](int kb) {
                if (kb >= kb_new && !waited) {
                    // buffer J & 1 was last read by the epilogue in panel J-2: done, since
                    // these producers passed xdone of panel J-2 in panel J-1
                    stage_b(J);
                    mbar_wait(xdone, (J - 1) & 1);   // panel J-1 solved and stored
                    waited = true;
                }
            };
            auto load = [&](float4 (&ra)[APER], float4 (&rb)[BPER], int kb) {
                ensure(kb);
                const int k0 = kb * BK;
#pragma unroll
                for (int p = 0; p < APER; p++) {
                    const int f = t + p * NP, row = f >> 3, c = f & 7;
                    ra[p] = (m0 + row < rows) ? ld_f4_cg(X + (int64_t)(m0 + row) * ldx + k0 + 4 * c) : z4;
                }
#pragma unroll
                for (int p = 0; p < BPER; p++) {
                    const int f = t + p * NP, row = f >> 3, c = f & 7;
                    const float *src = L + (int64_t)(c0 + row) * ldl + k0 + 4 * c;
                    rb[p] = (c0 + row < n) ? (POTRF ? ld_f4_cg(src) : __ldg(reinterpret_cast<const float4 *>(src))) : z4;
                }
            };
            auto produce = [&](float4 (&ra)[APER], float4 (&rb)[BPER], int kb) {
                const int s = gkb % STAGES;
                uint8_t *st = smem + s * G::STAGE;
                if (img) {
                    // POTRF: the k-block's split operands exist as images (stored by the rows'
                    // owners when they solved them): two bulk copies, no loads / splits here
                    ensure(kb);
                    if (t == 0) {
                        if (gkb >= STAGES) mbar_wait(&empty[s], ((gkb / STAGES) - 1) & 1);
                        fence_proxy_async_global();
                        const int nkb = n / BK;
                        img_expect_tx(&full[s], 2 * kImgKb);
                        img_g2s(smem_u32(st), img + ((size_t)blockIdx.x * nkb + kb) * kImgKb, kImgKb, &full[s]);
                        img_g2s(smem_u32(st) + kImgKb, img + ((size_t)J * nkb + kb) * kImgKb, kImgKb, &full[s]);
                    }
                } else {
                    if (gkb >= STAGES) mbar_wait(&empty[s], ((gkb / STAGES) - 1) & 1);
                    uint8_t *a_big = st, *a_small = st + G::A_BYTES;
                    uint8_t *b_big = st + 2 * G::A_BYTES, *b_small = b_big + G::B_BYTES;
#pragma unroll
                    for (int p = 0; p < APER; p++) {
                        const int f = t + p * NP, row = f >> 3, c = f & 7;
                        store_split(a_big, a_small, kmaj_off(row, c), ra[p]);
                    }
#pragma unroll
                    for (int p = 0; p < BPER; p++) {
                        const int f = t + p * NP, row = f >> 3, c = f & 7;
                        store_split(b_big, b_small, kmaj_off(row, c), rb[p]);
                    }
                    fence_proxy_async();
                    __syncwarp();
                    if (lane == 0) mbar_arrive(&full[s]);   // one release-arrive per producer warp
                }
                if (warp == 0) {
                    // MMA issue: all four producer warps have filled stage s
                    mbar_wait(&full[s], (gkb / STAGES) & 1);
                    tc_fence_after();
                    if (lane == 0) {
                        const uint32_t ab = smem_u32(st), as = ab + G::A_BYTES;
                        const uint32_t bb = ab + 2 * G::A_BYTES, bs = bb + G::B_BYTES;
#pragma unroll
                        for (int kk = 0; kk < BK / 8; kk++) {
                            uint64_t dAb, dAs, dBb, dBs;
                            if (img) {   // two SW64 halves of 16 k per part
                                const uint32_t o = (uint32_t)(kk >> 1) * kImgHalf + (uint32_t)(kk & 1) * 32;
                                dAb = desc_sw64(ab + o), dAs = desc_sw64(as + o);
                                dBb = desc_sw64(bb + o), dBs = desc_sw64(bs + o);
                            } else {
                                const uint32_t o = kk * 32;
                                dAb = make_desc(ab + o, 16, 1024), dAs = make_desc(as + o, 16, 1024);
                                dBb = make_desc(bb + o, 16, 1024), dBs = make_desc(bs + o, 16, 1024);
                            }
                            const uint32_t first = (kbp == 0 && kk == 0) ? 0u : 1u;
                            mma_tf32(dt, dAb, dBb, idesc, first);
                            mma_tf32(dt, dAb, dBs, idesc, 1u);
                            mma_tf32(dt, dAs, dBb, idesc, 1u);
                        }
                        mma_commit(&empty[s]);
                        if (kbp == nk - 1) mma_commit(&accf[J & 1]);
                        if (feed && J == fpanel && kbp == 0) {   // the accumulator is initialised
                            tc_fence_before();
                            mbar_arrive(pstart);
                        }
                    }
                    __syncwarp();
                }
                kbp++;
                gkb++;
            };
            float4 ra0[APER], rb0[BPER], ra1[APER], rb1[BPER];
            if (img) {
                for (int kb = 0; kb < nk; kb++) produce(ra0, rb0, kb);
            } else {
                load(ra0, rb0, 0);
                if (nk > 1) load(ra1, rb1, 1);
                for (int kb = 0; kb < nk; kb += 2) {
                    produce(ra0, rb0, kb);
                    if (kb + 2 < nk) load(ra0, rb0, kb + 2);
                    if (kb + 1 < nk) {
                        produce(ra1, rb1, kb + 1);
                        if (kb + 3 < nk) load(ra1, rb1, kb + 3);
                    }
                }
            }
            if (feed && J == fpanel) stage_b(J);   // (no k-block reached kb_new)
            if (t == 0) PANEL_T(J, 5);
        }
    } else {
        // =================================================== epilogue (warps 4-7)
        const int e = threadIdx.x - 128, row = m0 + e;
        const uint32_t tl = tmem + ((uint32_t)((warp & 3) * 32) << 16);
        const bool rowok = row < rows;
        float *xrow = X + (int64_t)(rowok ? row : 0) * ldx;
        uint32_t accn = 0;   // bit b: parity of the next accf[b] phase
        uint32_t xacc_par = 0;   // parity of the next xacc phase
        for (int J = 0; J < npanels; J++) {
            const int c0 = J * P, nk = c0 / BK, ncols = min(P, n - c0), nsb = ncols / PSB;
            const uint32_t acc = tl + (uint32_t)((J & 1) * P);
            const bool factor = POTRF && J == (int)blockIdx.x;
            bar_epi();   // Lt / colbuf of the previous panel no longer read
            if (!factor) {
                if (POTRF) {
                    if (e == 0) wait_flag(&flags[J], tag | (unsigned long long)(J + 1));
                    bar_epi();
                }
                if (e == 0) PANEL_T(J, 0);
                // stage L_JJ^T: rows q of L_JJ, coalesced in c = e; batched loads
#pragma unroll 1
                for (int q0 = 0; q0 < ncols; q0 += 32) {
                    float tmp[32];
#pragma unroll
                    for (int q = 0; q < 32; q++) {
                        const float *src = L + (int64_t)(c0 + q0 + q) * ldl + c0 + e;
                        tmp[q] = (e <= q0 + q && e < ncols) ? (POTRF ? ld_f_cg(src) : __ldg(src)) : 0.f;
                    }
#pragma unroll
                    for (int q = 0; q < 32; q++) Lt[e * LD + q0 + q] = tmp[q];
                }
                if (e < ncols) Lr[e] = rcp_approx(Lt[e * LD + e]);   // this thread's own store
                bar_epi();
                if (e == 0) PANEL_T(J, 1);
            }
            // b values of the panel (staged in TMEM by the producers)
            const uint32_t tbv = tl + (uint32_t)(2 * P + (J & 1) * P);
            mbar_wait(&bfull[J & 1], (uint32_t)(J >> 1) & 1u);
            // POTRF diagonal CTA: one dry pass of the sub-block body (no stores, no MMAs, no
            // info) while the panel's last MMAs run — the factor code runs only in this CTA's
            // last panel, and its first execution fetched ~25 KB of instructions from L2:
            // 2.3 us alone, 15 us under the GEMM flood (PANEL_T)
            const bool warm = factor && nk > 0 && (overlap & 2);
            auto acc_ready = [&]() {
                mbar_wait(&accf[J & 1], (accn >> (J & 1)) & 1u);
                accn ^= 1u << (J & 1);
                tc_fence_after();
                if (e == 0) PANEL_T(J, 2);
            };
            if (nk > 0) {
                if (!warm) acc_ready();
            } else {
                float z[16];
#pragma unroll
                for (int i = 0; i < 16; i++) z[i] = 0.f;
#pragma unroll 1
                for (int sb = 0; sb < nsb; sb++) tmem_st16(acc + sb * PSB, z);
            }
#pragma unroll 1
            for (int sbi = warm ? -1 : 0; sbi < nsb; sbi++) {
                const bool dry = sbi < 0;
                const int sb = dry ? 0 : sbi;
                if (warm && sbi == 0) acc_ready();
                float x[PSB], bv[PSB];
                tmem_ld16_issue(acc + sb * PSB, x);
                tmem_ld16_issue(tbv + sb * PSB, bv);
                tmem_wait_ld(x);
                tmem_wait_ld(bv);
#pragma unroll
                for (int i = 0; i < PSB; i++) x[i] = bv[i] - x[i];
                if (e == 0 && sbi == 0) PANEL_T(J, 22);
                if (factor) {
                    // the 16 x 16 diagonal sub-block is factored by the warp holding its rows,
                    // with shuffles (no block barrier per column); its L is published in Lt/Lr,
                    // then every row below solves against it exactly as the other CTAs' rows do
                    // (same operations and operands as a column-by-column right-looking sweep:
                    // l = sqrt(pivot), x_c = t_c / l by rcp + Newton, t_j -= x_c l_jc)
                    const int d0 = sb * PSB, lb = d0 & 31, r = e - d0;
                    const bool drow = r >= 0 && r < PSB;
                    if ((e >> 5) == (d0 >> 5)) {
                        float dg = 1.f;   // this row's diagonal l_rr (no dynamic index into x[])
#pragma unroll 16
                        for (int c = 0; c < PSB; c++) {
                            const float piv = __shfl_sync(0xffffffffu, x[c], lb + c);
                            const float l = sqrtf(piv);
                            // selects, not branches: under `r == c` the compiler would rewrite
                            // x[c] as x[r], a dynamic index that sends x[] to local memory
                            const bool piv_row = drow && r == c;
                            if (piv_row && !(piv > 0.f) && info && !dry) atomicCAS(info, 0, k_base + c0 + d0 + c + 1);
                            const float xd = div_nr(x[c], l, rcp_approx(l));
                            x[c] = piv_row ? l : ((drow && r > c) ? xd : x[c]);
                            dg = piv_row ? l : dg;
                            // rows below the pivot update every later column of the sub-block
                            // (entries right of their own diagonal are never stored)
                            const bool below = drow && r > c;
#pragma unroll 16
                            for (int j = 0; j < PSB; j++) {
                                if (j > c) {
                                    const float ljc = __shfl_sync(0xffffffffu, x[c], lb + j);
                                    const float upd = fmaf(-x[c], ljc, x[j]);
                                    x[j] = below ? upd : x[j];
                                }
                            }
                        }
                        if (drow && !dry) {
#pragma unroll
                            for (int c = 0; c < PSB; c++) Lt[(d0 + c) * LD + e] = x[c];
                            Lr[e] = rcp_approx(dg);
                        }
                    }
                    bar_epi();
                    if (r >= PSB) {
#pragma unroll
                        for (int c = 0; c < PSB; c++) {
                            const int cc = d0 + c;
                            x[c] = div_nr(x[c], Lt[cc * LD + cc], Lr[cc]);
#pragma unroll
                            for (int j = c + 1; j < PSB; j++) x[j] = fmaf(-x[c], Lt[cc * LD + d0 + j], x[j]);
                        }
                        // publish this row's L_JJ values (transposed) for the cross updates
                        if (!dry)
#pragma unroll
                            for (int c = 0; c < PSB; c++) Lt[(d0 + c) * LD + e] = x[c];
                    }
                    bar_epi();
                } else {
#pragma unroll
                    for (int c = 0; c < PSB; c++) {
                        const int cc = sb * PSB + c;
                        x[c] = div_nr(x[c], Lt[cc * LD + cc], Lr[cc]);
#pragma unroll
                        for (int j = c + 1; j < PSB; j++) x[j] = fmaf(-x[c], Lt[cc * LD + sb * PSB + j], x[j]);
                    }
                }
                if (e == 0 && sbi == 0) PANEL_T(J, 23);
                if (dry) continue;
                // store the solved row segment (diagonal block: lower part only)
                if (rowok) {
                    float *dst = xrow + c0 + sb * PSB;
                    if (factor) {
#pragma unroll
                        for (int c = 0; c < PSB; c++)
                            if (sb * PSB + c <= e) dst[c] = x[c];
                    } else {
#pragma unroll
                        for (int q = 0; q < PSB / 4; q++)
                            *reinterpret_cast<float4 *>(dst + 4 * q) =
                                make_float4(x[4 * q], x[4 * q + 1], x[4 * q + 2], x[4 * q + 3]);
                    }
                }
                // acc[:, later] += x_sb L[later, sb]^T for the later sub-blocks of the panel: one
                // tcgen05 3xTF32 MMA group (M = 128 rows, N = the later columns, K = 16) issued by
                // one epilogue thread into the panel's TMEM accumulator, operands staged in the
                // XS area (SW64 K-major: A = the 128 rows' 16 solved values, B = rows of L_JJ)
                if (e == 0) PANEL_T(J, 6 + 2 * sb);
                const bool feed_j = feed && J + 1 == fpanel;
                const bool need_img = img && !factor;   // operand image of a left-of-diagonal panel
                if (sb + 1 < nsb || feed_j || need_img) {
                    const int nb = (nsb - sb - 1) * PSB;   // later columns (a multiple of 16)
                    {   // A: this row's values, split big / small
                        const uint32_t ra = (uint32_t)e * 64u;
#pragma unroll
                        for (int q = 0; q < 4; q++) {
                            const uint32_t off = ra + ((uint32_t)(q ^ ((e >> 1) & 3)) << 4);
                            store_split(xs_ab, xs_as, off, make_float4(x[4 * q], x[4 * q + 1], x[4 * q + 2], x[4 * q + 3]));
                        }
                    }
                    if (e < nb && sb + 1 < nsb) {   // B: row (sb+1)*16 + e of L_JJ, columns sb*16 .. +15 (from Lt)
                        const float *lc = Lt + (sb * PSB) * LD + (sb + 1) * PSB + e;
                        const uint32_t rb = (uint32_t)e * 64u;
#pragma unroll
                        for (int q = 0; q < 4; q++) {
                            const float4 v = make_float4(lc[(4 * q) * LD], lc[(4 * q + 1) * LD], lc[(4 * q + 2) * LD],
                                                         lc[(4 * q + 3) * LD]);
                            store_split(xs_bb, xs_bs, rb + ((uint32_t)(q ^ ((e >> 1) & 3)) << 4), v);
                        }
                    }
                    fence_proxy_async();
                    tc_fence_before();
                    bar_epi();
                    if (e == 0) {
                        tc_fence_after();
                        const uint32_t ab = smem_u32(xs_ab), as = smem_u32(xs_as), bb = smem_u32(xs_bb), bs = smem_u32(xs_bs);
                        if (need_img) {   // the staged split x block is the image's half sb & 1
                            const int nkb = n / BK;
                            uint8_t *ib = img + ((size_t)blockIdx.x * nkb + (c0 + sb * PSB) / BK) * kImgKb + (sb & 1) * kImgHalf;
                            img_s2g(ib, ab, kImgHalf);
                            img_s2g(ib + 2 * kImgHalf, as, kImgHalf);
                            img_commit();
                        }
                        if (sb + 1 < nsb) {
                            const uint32_t idesc = make_idesc(BM, nb, false, false);
                            const uint32_t d = tmem + (uint32_t)((J & 1) * P + (sb + 1) * PSB);
#pragma unroll
                            for (int kk = 0; kk < PSB / 8; kk++) {
                                const uint32_t o = kk * 32;
                                mma_tf32(d, desc_sw64(ab + o), desc_sw64(bb + o), idesc, 1u);
                                mma_tf32(d, desc_sw64(ab + o), desc_sw64(bs + o), idesc, 1u);
                                mma_tf32(d, desc_sw64(as + o), desc_sw64(bb + o), idesc, 1u);
                            }
                        }
                        if (feed_j) {
                            // acc[factor panel] += x_sb x_sb^T: these rows are the factor panel's
                            // rows and columns (A = B = the staged x block), after the producers'
                            // first (initialising) MMA of that panel
                            if (sb == 0 && feed_pk) {
                                mbar_wait(pstart, 0);
                                tc_fence_after();
                            }
                            const uint32_t idesc = make_idesc(BM, P, false, false);
                            const uint32_t d = tmem + (uint32_t)(((J + 1) & 1) * P);
#pragma unroll
                            for (int kk = 0; kk < PSB / 8; kk++) {
                                const uint32_t o = kk * 32;
                                const uint32_t init = (!feed_pk && sb == 0 && kk == 0) ? 0u : 1u;
                                mma_tf32(d, desc_sw64(ab + o), desc_sw64(ab + o), idesc, init);
                                mma_tf32(d, desc_sw64(ab + o), desc_sw64(as + o), idesc, 1u);
                                mma_tf32(d, desc_sw64(as + o), desc_sw64(ab + o), idesc, 1u);
                            }
                        }
                        if (sb + 1 < nsb || feed_j) mma_commit(xacc);
                        else mbar_arrive(xacc);
                        if (need_img) img_wait_read();   // the staged block may be overwritten
                        mbar_arrive(xacc);
                    }
                    mbar_wait(xacc, xacc_par);
                    xacc_par ^= 1u;
                    tc_fence_after();
                }
                if (e == 0) PANEL_T(J, 7 + 2 * sb);
            }
            if (e == 0) PANEL_T(J, 3);
            if (img && !factor && e == 0) {   // the panel's images written before xdone / the flag
                img_wait_all();
                fence_proxy_async_global();
            }
            // panel J of these rows: visible at L2 (own producers, other CTAs), TMEM reads done
            __threadfence();
            tc_fence_before();
            __syncwarp();
            if (lane == 0) mbar_arrive(xdone);
            if (POTRF) {
                bar_epi();
                if (e == 0) st_release(&flags[blockIdx.x], tag | (unsigned long long)(J + 1));
            }
        }
    }

    tc_fence_before();
    __syncthreads();
    tc_fence_after();
    if (warp == 0) {
        asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"((uint32_t)(4 * P)));
    }
    ctx_end(ctx);
}

// kernel option bits (measurement switches): bit 0 — MMA of panel J+1 overlapped with the
// solve of panel J (default; VS_PANEL_OVERLAP=0 serialises them); bit 1 — the diagonal CTA's
// dry pass of the factor code (default; VS_PANEL_WARM=0 disables); bit 2 — POTRF feed of the
// factor panel's accumulator by the previous panel's solve (default; VS_PANEL_FEED=0 disables);
// bit 3 — POTRF operand images (default; VS_PANEL_IMG=0: the producers load and split)
inline int panel_overlap()
{
    static const int v = [] {
        const char *e = getenv("VS_PANEL_OVERLAP");
        const char *w = getenv("VS_PANEL_WARM");
        const char *f = getenv("VS_PANEL_FEED");
        const char *im = getenv("VS_PANEL_IMG");
        return (e ? (atoi(e) ? 1 : 0) : 1) | ((w ? (atoi(w) ? 1 : 0) : 1) << 1) | ((f ? (atoi(f) ? 1 : 0) : 1) << 2) |
               ((im ? (atoi(im) ? 1 : 0) : 1) << 3);
    }();
    return v;
}

template <bool POTRF>
inline void panel_attr()
{
    static bool attr[64] = {};
    int dev = 0;
    cudaGetDevice(&dev);
    if (!attr[dev & 63]) {
        cudaFuncSetAttribute(tc_panel_kernel<POTRF>, cudaFuncAttributeMaxDynamicSharedMemorySize, PanelCfg::SMEM);
        attr[dev & 63] = true;
    }
}

// X <- X L^{-T}: rows x n (n % 64 == 0), one launch.
inline int tc_trsm(int rows, int n, const float *L, int ldl, float *X, int ldx, cudaStream_t s,
                   const TaskCtx &ctx = TaskCtx())
{
    if (rows <= 0 || n <= 0) return 0;
    if (n % 64) return -1;
    panel_attr<false>();
    count_launch();
    tc_panel_kernel<false><<<(rows + BM - 1) / BM, PTHREADS, PanelCfg::SMEM, s>>>(rows, n, L, ldl, X, ldx, 0, nullptr,
                                                                                  0ull, panel_overlap(), 0, 0, ctx, nullptr);
    return 0;
}

// count independent X_i <- X_i L_i^{-T} (X_i = X + i xbs, L_i = L + i lbs), one launch.
inline int tc_trsm_batched(int count, int rows, int n, const float *L, int ldl, int64_t lbs, float *X, int ldx,
                           int64_t xbs, cudaStream_t s)
{
    if (rows <= 0 || n <= 0 || count <= 0) return 0;
    if (n % 64) return -1;
    panel_attr<false>();
    count_launch();
    tc_panel_kernel<false><<<dim3((rows + BM - 1) / BM, count), PTHREADS, PanelCfg::SMEM, s>>>(
        rows, n, L, ldl, X, ldx, 0, nullptr, 0ull, panel_overlap(), lbs, xbs, TaskCtx(), nullptr);
    return 0;
}

// A = L L^T in place: n x n (n % 64 == 0, n <= 4096), one launch.
inline int tc_potrf(int n, float *A, int lda, int k_base, int *info, cudaStream_t s, const TaskCtx &ctx = TaskCtx())
{
    if (n <= 0) return 0;
    if (n % 64 || (n + BM - 1) / BM > kFlagCtas) return -1;
    static std::atomic<unsigned long long> next_id{1};
    const unsigned long long id = next_id.fetch_add(1);
#ifdef VS_PANEL_TRACE
    // one potrf of a whole run (VS_TRACE_POTRF = its launch id), dumped at exit to VS_TRACE_FILE
    static const unsigned long long want = [] {
        const char *e = getenv("VS_TRACE_POTRF");
        const unsigned long long w = e ? strtoull(e, nullptr, 10) : 0;
        cudaMemcpyToSymbol(g_panel_trace_id, &w, sizeof w);
        if (w) atexit([] {
            static unsigned long long tr[32][32][24];
            static long long ck[32][32][24];
            cudaDeviceSynchronize();
            cudaMemcpyFromSymbol(tr, g_panel_trace, sizeof tr);
            cudaMemcpyFromSymbol(ck, g_panel_clk, sizeof ck);
            const char *f = getenv("VS_TRACE_FILE");
            if (FILE *fp = fopen(f ? f : "panel_trace.bin", "wb")) {
                fwrite(tr, sizeof tr, 1, fp);
                fwrite(ck, sizeof ck, 1, fp);
                fclose(fp);
            }
        });
        return w;
    }();
    (void)want;
#endif
    panel_attr<true>();
    count_launch();
    const int grid = (n + BM - 1) / BM;
    // operand images (option bit 3, VS_PANEL_IMG): stream-ordered scratch from the device's
    // default memory pool (its release threshold raised once, so the pool keeps the memory)
    uint8_t *img = nullptr;
    if ((panel_overlap() & 8) && n >= 1024) {   // b = 512: 190 vs 183 us with images (4 panels)
        static bool pool_set[64] = {};
        int dev = 0;
        cudaGetDevice(&dev);
        cudaStreamCaptureStatus cs = cudaStreamCaptureStatusNone;
        cudaStreamIsCapturing(s, &cs);
        if (!pool_set[dev & 63] && cs == cudaStreamCaptureStatusNone) {
            cudaMemPool_t pool;
            if (cudaDeviceGetDefaultMemPool(&pool, dev) == cudaSuccess) {
                unsigned long long thr = ~0ull;
                cudaMemPoolSetAttribute(pool, cudaMemPoolAttrReleaseThreshold, &thr);
            }
            pool_set[dev & 63] = true;
        }
        if (cudaMallocAsync((void **)&img, (size_t)grid * (n / BK) * kImgKb, s) != cudaSuccess) {
            cudaGetLastError();
            img = nullptr;   // the loads-and-splits producers
        }
    }
    tc_panel_kernel<true><<<grid, PTHREADS, PanelCfg::SMEM, s>>>(n, n, A, lda, A, lda, k_base, info, id,
                                                                 panel_overlap(), 0, 0, ctx, img);
    if (img) cudaFreeAsync(img, s);
    return 0;
}

}  // namespace tc
}  // namespace vsk
