// builtin.cu — the built-in tile task versions (VS_T_* x VS_V_*): each version is a
// sequence of sm_100a kernels enqueued on the worker's stream.  Every kernel receives the
// task's TaskCtx (task_ctx.cuh) so the task's GPU execution interval is recorded on the
// device.
//
//   version        storage  GEMM engine (matmul/gemm/syrk + potrf/trsm updates)   trsm
//   simt_f32       fp32     simt_gemm<float,float>   (FFMA, bit-exact Fig 1 order)  blocked
//   tc_3xtf32      fp32     tc_gemm (tcgen05/TMEM 3xTF32)                          tc_panel (1 launch)
//   f64in_f32io    fp32     dmma_gemm<float>  (DMMA on upcast operands)            blocked
//   dfma_f64       fp64     simt_gemm<double,double> (DFMA)                        blocked
//   dmma_f64       fp64     dmma_gemm<double>  (mma.sync f64)                      blocked
//   tc_3xf16       fp32     tcf_gemm (tcgen05 kind::f16 on split forms, tc_f16.cuh); TRSM = GEMM with
//                           the inv(L) form (R31); no potrf
//   oz_i8_f64      fp64     oz_gemm (tcgen05 kind::i8 Ozaki scheme on slice forms, tc_oz.cuh);
//                           MATMUL / GEMM_NT / SYRK only
//
// potrf of tc_3xtf32 is the single-launch left-looking tc_panel kernel (tc_panel.cuh).
// potrf of the other versions is recursive: potrf(A11); A21 <- A21 L11^{-T} (trsm);
// A22 -= A21 A21^T (lower GEMM); potrf(A22), down to an NB x NB diagonal block factored
// in registers (simt_chol.cuh).  Blocked trsm: NB-wide panels solved by trsm_panel,
// remaining columns updated by the engine's GEMM.
#include <map>
#include <mutex>
#include <tuple>
#include <type_traits>

#include "blk_chol.cuh"
#include "dmma_gemm.cuh"
#include "kernels.hpp"
#include "simt_chol.cuh"
#include "simt_gemm.cuh"
#include "tc_gemm.cuh"
#include "tc_f16.cuh"
#include "tc_oz.cuh"
#include "tc_inv.cuh"
#include "tc_panel.cuh"

#include "vsched.h"

namespace vsk {

namespace {

__global__ void eye64_kernel(double *X, int n)
{
    for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < (int64_t)n * n; i += (int64_t)gridDim.x * blockDim.x)
        X[i] = (i / n == i % n) ? 1.0 : 0.0;
}

template <typename Tin, typename Tp, class Gemm>
int blocked_trsm(int rows, int n, const Tin *L, int ldl, Tin *X, int ldx, cudaStream_t s, const TaskCtx &ctx)
{
    constexpr int NBP = sizeof(Tp) == 4 ? 64 : 32;
    for (int j0 = 0; j0 < n; j0 += NBP) {
        trsm_panel<Tin, Tp, NBP>(L + (int64_t)j0 * ldl + j0, ldl, X + j0, ldx, rows, s, ctx);
        const int rest = n - j0 - NBP;
        if (rest > 0) {
            int r = Gemm::template gemm<true, true, false>(rows, rest, NBP, X + j0, ldx, L + (int64_t)(j0 + NBP) * ldl + j0,
                                                           ldl, X + j0 + NBP, ldx, s, ctx);
            if (r) return r;
        }
    }
    return 0;
}

template <typename Tin, typename Tacc>
struct SimtEngine {
    using Tp = Tacc;
    template <bool NT, bool NEG, bool LOWER>
    static int gemm(int M, int N, int K, const Tin *A, int lda, const Tin *B, int ldb, Tin *C, int ldc, cudaStream_t s,
                    const TaskCtx &ctx)
    {
        simt_gemm<Tin, Tacc, NT, NEG, LOWER>(M, N, K, A, lda, B, ldb, C, ldc, s, ctx);
        return 0;
    }
    static int trsm(int rows, int n, const Tin *L, int ldl, Tin *X, int ldx, cudaStream_t s, const TaskCtx &ctx)
    {
        if constexpr (std::is_same<Tin, float>::value && std::is_same<Tacc, float>::value)
            return blk::trsm(rows, n, L, ldl, X, ldx, s, ctx);   // one launch, sub-tile DAG (blk_chol.cuh)
        else
            return blocked_trsm<Tin, Tp, SimtEngine>(rows, n, L, ldl, X, ldx, s, ctx);
    }
};
template <typename Tin>
struct DmmaEngine {
    using Tp = double;
    template <bool NT, bool NEG, bool LOWER>
    static int gemm(int M, int N, int K, const Tin *A, int lda, const Tin *B, int ldb, Tin *C, int ldc, cudaStream_t s,
                    const TaskCtx &ctx)
    {
        dmma_gemm<Tin, NT, NEG, LOWER>(M, N, K, A, lda, B, ldb, C, ldc, s, ctx);
        return 0;
    }
    static int trsm(int rows, int n, const Tin *L, int ldl, Tin *X, int ldx, cudaStream_t s, const TaskCtx &ctx)
    {
        return blocked_trsm<Tin, Tp, DmmaEngine>(rows, n, L, ldl, X, ldx, s, ctx);
    }
};
// oz_i8_f64 POTRF (recursive, like the DFMA / DMMA versions): the trailing updates are Ozaki-
// scheme tcgen05 kind::i8 GEMMs on slice forms built per call in stream-ordered scratch; the
// panel trsm is the blocked DMMA substitution, the diagonal blocks the DFMA register kernel.
struct OzEngine {
    using Tp = double;
    template <bool NT, bool NEG, bool LOWER>
    static int gemm(int M, int N, int K, const double *A, int lda, const double *B, int ldb, double *C, int ldc,
                    cudaStream_t s, const TaskCtx &ctx)
    {
        static_assert(NT && NEG, "potrf_rec only needs C -= A B^T");
        if (M <= 0 || N <= 0 || K <= 0) return 0;
        // the small updates near the recursion's leaves stay on DMMA (slice forms need K % 64,
        // N % 64, and do not pay off below 128)
        if (K % 64 || N % oz::BN || M < 128 || N < 128 || K < 128 || (LOWER && M != N))
            return DmmaEngine<double>::template gemm<NT, NEG, LOWER>(M, N, K, A, lda, B, ldb, C, ldc, s, ctx);
        const size_t fa = (oz::form_bytes(M, K) + 255) / 256 * 256;
        const size_t fb = LOWER ? 0 : (oz::form_bytes(N, K) + 255) / 256 * 256;
        void *buf = nullptr;
        if (cudaMallocAsync(&buf, fa + fb, s) != cudaSuccess) return -1;
        uint8_t *pa = (uint8_t *)buf, *pb = LOWER ? pa : pa + fa;
        int r = oz::make_slices(A, M, K, lda, 1, 128, pa, s, true);
        if (!r && !LOWER) r = oz::make_slices(B, N, K, ldb, 1, 64, pb, s, true);
        if (!r) r = LOWER ? oz::oz_gemm<true, true, 128>(M, N, K, pa, pb, C, ldc, s, false, ctx)
                          : oz::oz_gemm<true, false, 64>(M, N, K, pa, pb, C, ldc, s, false, ctx);
        cudaFreeAsync(buf, s);
        return r;
    }
    static int trsm(int rows, int n, const double *L, int ldl, double *X, int ldx, cudaStream_t s, const TaskCtx &ctx)
    {
        return DmmaEngine<double>::trsm(rows, n, L, ldl, X, ldx, s, ctx);
    }
};

struct TcEngine {
    using Tp = float;
    template <bool NT, bool NEG, bool LOWER>
    static int gemm(int M, int N, int K, const float *A, int lda, const float *B, int ldb, float *C, int ldc,
                    cudaStream_t s, const TaskCtx &ctx)
    {
        return tc::tc_gemm<NT, NEG, LOWER>(M, N, K, A, lda, B, ldb, C, ldc, s, ctx);
    }
    // single-launch left-looking panel kernel (tc_panel.cuh)
    static int trsm(int rows, int n, const float *L, int ldl, float *X, int ldx, cudaStream_t s, const TaskCtx &ctx)
    {
        return tc::tc_trsm(rows, n, L, ldl, X, ldx, s, ctx);
    }
};

// Recursive Cholesky of the n x n lower block at A (leading dimension ld), global column
// offset k_base (for info).
template <typename Tin, class E>
int potrf_rec(Tin *A, int n, int ld, int k_base, int *info, cudaStream_t s, const TaskCtx &ctx)
{
    using Tp = typename E::Tp;
    constexpr int NBP = sizeof(Tp) == 4 ? 64 : 32;
    if (n <= NBP) {
        potrf_diag<Tin, Tp, NBP>(A, ld, k_base, info, s, ctx);
        return 0;
    }
    int h = (n / 2) / 64 * 64;
    if (h < NBP) h = NBP;
    const int r = n - h;
    Tin *A21 = A + (int64_t)h * ld, *A22 = A + (int64_t)h * ld + h;
    int rc = potrf_rec<Tin, E>(A, h, ld, k_base, info, s, ctx);
    if (!rc) rc = E::trsm(r, h, A, ld, A21, ld, s, ctx);
    if (!rc) rc = E::template gemm<true, true, true>(r, r, h, A21, ld, A21, ld, A22, ld, s, ctx);
    if (!rc) rc = potrf_rec<Tin, E>(A22, r, ld, k_base + h, info, s, ctx);
    return rc;
}

// Tin = storage, E = engine.
template <typename Tin, class E>
int run_family(int type, int b, void *const *p, int *info, cudaStream_t s, const TaskCtx &ctx)
{
    switch (type) {
    case VS_T_MATMUL:  // C += A B                 (Fig 1)
        return E::template gemm<false, false, false>(b, b, b, (const Tin *)p[0], b, (const Tin *)p[1], b, (Tin *)p[2], b,
                                                     s, ctx);
    case VS_T_GEMM_NT:  // C -= A B^T              (R5)
        return E::template gemm<true, true, false>(b, b, b, (const Tin *)p[0], b, (const Tin *)p[1], b, (Tin *)p[2], b,
                                                   s, ctx);
    case VS_T_SYRK:  // C -= A A^T, lower          (R5, R7)
        return E::template gemm<true, true, true>(b, b, b, (const Tin *)p[0], b, (const Tin *)p[0], b, (Tin *)p[1], b, s,
                                                  ctx);
    case VS_T_TRSM:  // B <- B L^{-T}              (R5)
        return E::trsm(b, b, (const Tin *)p[0], b, (Tin *)p[1], b, s, ctx);
    case VS_T_POTRF:  // A = L L^T in place        (L697-699, R9)
        if constexpr (std::is_same<E, TcEngine>::value)
            return tc::tc_potrf(b, (float *)p[0], b, 0, info, s, ctx);   // single launch (tc_panel.cuh)
        else if constexpr (std::is_same<E, SimtEngine<float, float>>::value)
            return blk::potrf(b, (float *)p[0], b, 0, info, s, ctx);     // single launch (blk_chol.cuh)
        else
            return potrf_rec<Tin, E>((Tin *)p[0], b, b, 0, info, s, ctx);
    }
    return -1;
}

}  // namespace

int builtin_elem_bytes(int version)
{
    return (version == VS_V_DFMA_F64 || version == VS_V_DMMA_F64 || version == VS_V_OZ_I8_F64) ? 8 : 4;
}

bool builtin_supported(int type, int version, int b)
{
    if (type < 0 || type >= VS_NUM_BUILTIN_TYPES) return false;
    if (version < 0 || version >= VS_NUM_BUILTIN_VERSIONS) return false;
    if (version == VS_V_TC_3XF16 && type == VS_T_POTRF) return false;
    if (b && (b % 64 != 0 || b < 64 || b > 4096)) return false;
    return true;
}

int builtin_nparams(int type)
{
    static const int np[VS_NUM_BUILTIN_TYPES] = {3, 1, 2, 2, 3};
    return (type >= 0 && type < VS_NUM_BUILTIN_TYPES) ? np[type] : 0;
}

int builtin_operand_form(int type, int version, int param)
{
    if (version == VS_V_OZ_I8_F64) {
        switch (type) {
        case VS_T_MATMUL: return param == 0 ? FORM_OZ_ROWS : param == 1 ? FORM_OZ_COLS : FORM_RAW;
        case VS_T_GEMM_NT: return param == 0 ? FORM_OZ_ROWS : param == 1 ? FORM_OZ_ROWS_B : FORM_RAW;
        case VS_T_SYRK: return param == 0 ? FORM_OZ_ROWS : FORM_RAW;
        case VS_T_TRSM: return param == 0 ? FORM_OZ_INV_L : FORM_OZ_ROWS;   // X = B inv(L)^T
        }
        return FORM_RAW;
    }
    if (version != VS_V_TC_3XF16) return FORM_RAW;
    switch (type) {
    case VS_T_MATMUL: return param == 0 ? FORM_SPLIT_ROWS : param == 1 ? FORM_SPLIT_COLS : FORM_RAW;
    case VS_T_GEMM_NT: return param <= 1 ? FORM_SPLIT_ROWS : FORM_RAW;
    case VS_T_SYRK: return param == 0 ? FORM_SPLIT_ROWS : FORM_RAW;
    case VS_T_TRSM: return param == 0 ? FORM_INV_L : param == 1 ? FORM_SPLIT_ROWS : FORM_RAW;   // X = B inv(L)^T
    }
    return FORM_RAW;
}

size_t form_bytes(int form, int b)
{
    if (form == FORM_RAW) return 0;
    if (form == FORM_OZ_ROWS || form == FORM_OZ_COLS || form == FORM_OZ_ROWS_B)
        return (oz::form_bytes(b, b) + 255) / 256 * 256;
    if (form == FORM_OZ_INV_L) return (oz::form_bytes(b, b) + 255) / 256 * 256 + (size_t)b * b * 8;   // + fp64 scratch
    const size_t sb = (tcf::split_bytes(b, b) + 255) / 256 * 256;
    return form == FORM_INV_L ? sb + (size_t)b * b * 4 : sb;   // + fp32 scratch for inv(L)^T
}

int make_form(int form, int b, const void *src, void *dst, cudaStream_t s)
{
    if (form == FORM_OZ_ROWS) return oz::make_slices((const double *)src, b, b, b, 1, 128, dst, s);
    if (form == FORM_OZ_ROWS_B) return oz::make_slices((const double *)src, b, b, b, 1, 64, dst, s);
    if (form == FORM_OZ_COLS) return oz::make_slices((const double *)src, b, b, 1, b, 64, dst, s);
    if (form == FORM_OZ_INV_L) {
        // X = I L^{-T} (fp64, the blocked DMMA substitution of dmma_f64), then the slice form of
        // the columns of X = the rows of inv(L) in the B role
        double *X = (double *)((uint8_t *)dst + (oz::form_bytes(b, b) + 255) / 256 * 256);
        count_launch();
        eye64_kernel<<<148, 256, 0, s>>>(X, b);
        if (DmmaEngine<double>::trsm(b, b, (const double *)src, b, X, b, s, TaskCtx())) return -1;
        return oz::make_slices(X, b, b, 1, b, 64, dst, s);
    }
    if (form == FORM_SPLIT_ROWS) return tcf::split_rows((const float *)src, b, b, b, dst, s);
    if (form == FORM_SPLIT_COLS) return tcf::split_cols((const float *)src, b, b, b, dst, s);
    if (form == FORM_INV_L) {
        // X = L^{-T} by recursive doubling on the 3xTF32 kernels (tc_inv.cuh; the whole-tile
        // substitution of tc_panel took 258 us at b = 1024, the sub-tile DAG of blk_chol.cuh
        // 719 us), then the row split form of X^T = inv(L): reading R31 (TRSM of tc_3xf16
        // multiplies by it).  The split area is the recursion's scratch until split_cols.
        float *X = (float *)((uint8_t *)dst + (tcf::split_bytes(b, b) + 255) / 256 * 256);
        count_launch();
        tcf::eye_kernel<<<148, 256, 0, s>>>(X, b);
        if (tc::tc_inv_lt(b, (const float *)src, b, X, b, (float *)dst, s)) return -1;
        return tcf::split_cols(X, b, b, b, dst, s);
    }
    return -1;
}

struct TaskGroup {
    tcf::TcfGroup g;
};
int group_kind(int type, int version, int b)
{
    // a tile whose K needs several accumulation chunks (tc::kKChunk) runs as sequential
    // launches, never inside a group
    return (version == VS_V_TC_3XF16 && type != VS_T_POTRF && b <= tc::kKChunk) ? 1 : 0;
}
TaskGroup *group_new() { return new TaskGroup(); }
void group_free(TaskGroup *g) { delete g; }
int group_size(const TaskGroup *g) { return g->g.n; }
int group_ctas(const TaskGroup *g) { return g->g.ctas; }
// the K-chunk [k0, k0 + kc) of one tc_3xf16 task (kc < 0: all of K)
static int group_add_chunk(TaskGroup *g, int type, int b, void *const *p, const TaskCtx &ctx, int k0, int kc)
{
    switch (type) {   // p[i] tiles, p[np + i] forms (np = 3 / 2 / 2)
    case VS_T_MATMUL: return tcf::tcf_group_add(g->g, b, b, b, p[3], p[4], (float *)p[2], b, false, false, ctx, false, k0, kc);
    case VS_T_GEMM_NT: return tcf::tcf_group_add(g->g, b, b, b, p[3], p[4], (float *)p[2], b, true, false, ctx, false, k0, kc);
    case VS_T_SYRK: return tcf::tcf_group_add(g->g, b, b, b, p[2], p[2], (float *)p[1], b, true, true, ctx, false, k0, kc);
    case VS_T_TRSM:   // X = B inv(L)^T: C_in not read by the first chunk
        return tcf::tcf_group_add(g->g, b, b, b, p[3], p[2], (float *)p[1], b, false, false, ctx, k0 == 0, k0, kc);
    }
    return -1;
}
int group_add(TaskGroup *g, int type, int version, int b, void *const *p, const TaskCtx &ctx)
{
    if (!group_kind(type, version, b)) return -1;
    return group_add_chunk(g, type, b, p, ctx, 0, -1);
}
int group_launch(TaskGroup *g, cudaStream_t s) { return tcf::tcf_group_launch(g->g, s); }

namespace {
// oz_i8_f64: p[np + i] holds the slice forms of the in-operands (builtin_operand_form)
int run_oz(int type, int b, void *const *p, int *info, cudaStream_t s, const TaskCtx &ctx)
{
    switch (type) {
    case VS_T_POTRF: return potrf_rec<double, OzEngine>((double *)p[0], b, b, 0, info, s, ctx);   // A = L L^T
    case VS_T_MATMUL: return oz::oz_gemm<false, false, 64>(b, b, b, p[3], p[4], (double *)p[2], b, s, false, ctx);   // C += A B
    case VS_T_GEMM_NT: return oz::oz_gemm<true, false, 64>(b, b, b, p[3], p[4], (double *)p[2], b, s, false, ctx);  // C -= A B^T
    case VS_T_SYRK: return oz::oz_gemm<true, true, 128>(b, b, b, p[2], p[2], (double *)p[1], b, s, false, ctx);   // C -= A A^T
    case VS_T_TRSM: return oz::oz_gemm<false, false, 64>(b, b, b, p[3], p[2], (double *)p[1], b, s, true, ctx);  // X = B inv(L)^T
    }
    return -1;
}
// tc_3xf16: p[] holds the split forms of the in-operands (builtin_operand_form)
int run_f16(int type, int b, void *const *p, cudaStream_t s, const TaskCtx &ctx)
{
    if (type == VS_T_POTRF) return -1;
    for (int k0 = 0; k0 < b; k0 += tc::kKChunk) {   // accumulation accuracy: see tc::tc_gemm
        TaskGroup g;
        const int r = group_add_chunk(&g, type, b, p, ctx, k0, b - k0 < tc::kKChunk ? b - k0 : tc::kKChunk);
        if (r <= 0) return r;
        if (group_launch(&g, s)) return -1;
    }
    return 0;
}
}  // namespace

int builtin_kernel_count(int type, int version, int b)
{
    static std::mutex mu;
    static std::map<std::tuple<int, int, int>, int> cache;
    if (!builtin_supported(type, version, b)) return -1;
    std::lock_guard<std::mutex> lock(mu);
    const auto key = std::make_tuple(type, version, b);
    auto it = cache.find(key);
    if (it != cache.end()) return it->second;
    // capture one launch into a graph (nothing executes; pointers are never dereferenced)
    cudaStream_t st = nullptr;
    if (cudaStreamCreateWithFlags(&st, cudaStreamNonBlocking) != cudaSuccess) return -1;
    void *fake[8];
    for (int i = 0; i < 8; i++) fake[i] = (void *)(uintptr_t)(0x100000 * (i + 1));
    int n = -1;
    const long long c0 = launch_counter().load();
    if (cudaStreamBeginCapture(st, cudaStreamCaptureModeThreadLocal) == cudaSuccess) {
        const int r = launch_builtin(type, version, b, fake, (int *)fake[7], st);
        cudaGraph_t g = nullptr;
        const bool ok = cudaStreamEndCapture(st, &g) == cudaSuccess && r == 0;
        if (ok) n = (int)(launch_counter().load() - c0);
        if (g) cudaGraphDestroy(g);
    }
    launch_counter().fetch_sub(launch_counter().load() - c0);   // captured, never launched
    cudaGetLastError();
    cudaStreamDestroy(st);
    if (n >= 0) cache[key] = n;
    return n;
}

int launch_release(const TaskCtx &ctx, cudaStream_t s)
{
    if (!ctx.trk) return 0;
    count_launch();
    release_kernel<<<1, 32, 0, s>>>(ctx);
    return cudaGetLastError() == cudaSuccess ? 0 : -1;
}

int launch_builtin(int type, int version, int b, void *const *p, int *info, cudaStream_t s, const TaskCtx &ctx)
{
    if (!builtin_supported(type, version, b)) return -1;
    switch (version) {
    case VS_V_SIMT_F32: return run_family<float, SimtEngine<float, float>>(type, b, p, info, s, ctx);
    case VS_V_TC_3XTF32: return run_family<float, TcEngine>(type, b, p, info, s, ctx);
    case VS_V_F64IN_F32IO: return run_family<float, DmmaEngine<float>>(type, b, p, info, s, ctx);
    case VS_V_DFMA_F64: return run_family<double, SimtEngine<double, double>>(type, b, p, info, s, ctx);
    case VS_V_DMMA_F64: return run_family<double, DmmaEngine<double>>(type, b, p, info, s, ctx);
    case VS_V_TC_3XF16: return run_f16(type, b, p, s, ctx);
    case VS_V_OZ_I8_F64: return run_oz(type, b, p, info, s, ctx);
    }
    return -1;
}

}  // namespace vsk

#ifdef VS_TCF_TRACE
// measurement builds only: read (and reset) the tc_3xf16 GEMM's per-CTA phase records
extern "C" __attribute__((visibility("default"))) int vs_debug_tcf_trace(unsigned long long *out, int cap)
{
    unsigned int n = 0;
    cudaDeviceSynchronize();
    cudaMemcpyFromSymbol(&n, vsk::tcf::g_tcf_n, sizeof n);
    if (n > (unsigned)vsk::tcf::kTcfTraceCap) n = vsk::tcf::kTcfTraceCap;
    if (n > (unsigned)cap) n = (unsigned)cap;
    if (n) cudaMemcpyFromSymbol(out, vsk::tcf::g_tcf_rec, (size_t)n * 12 * sizeof(unsigned long long));
    unsigned int z = 0;
    cudaMemcpyToSymbol(vsk::tcf::g_tcf_n, &z, sizeof z);
    return (int)n;
}
#endif
