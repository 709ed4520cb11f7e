// builtin.cu — the built-in tile task versions (VS_T_* x VS_V_*): each version is a
// sequence of sm_100a kernels enqueued on the worker's stream.
//
//   version        storage  GEMM engine (matmul/gemm/syrk + potrf/trsm updates)   panels
//   simt_f32       fp32     simt_gemm<float,float>   (FFMA, bit-exact Fig 1 order)  fp32
//   tc_3xtf32      fp32     tc_gemm (tcgen05/TMEM 3xTF32)                          fp32
//   f64in_f32io    fp32     dmma_gemm<float>  (DMMA on upcast operands)            fp64
//   dfma_f64       fp64     simt_gemm<double,double> (DFMA)                        fp64
//   dmma_f64       fp64     dmma_gemm<double>  (mma.sync f64)                      fp64
#include "dmma_gemm.cuh"
#include "kernels.hpp"
#include "simt_chol.cuh"
#include "simt_gemm.cuh"
#include "tc_gemm.cuh"

#include "vsched.h"

namespace vsk {

namespace {

template <typename Tin, typename Tacc>
struct SimtEngine {
    template <bool NT, bool NEG, bool LOWER>
    static int gemm(int M, int N, int K, const Tin *A, int lda, const Tin *B, int ldb, Tin *C, int ldc, cudaStream_t s)
    {
        simt_gemm<Tin, Tacc, NT, NEG, LOWER>(M, N, K, A, lda, B, ldb, C, ldc, s);
        return 0;
    }
};
template <typename Tin>
struct DmmaEngine {
    template <bool NT, bool NEG, bool LOWER>
    static int gemm(int M, int N, int K, const Tin *A, int lda, const Tin *B, int ldb, Tin *C, int ldc, cudaStream_t s)
    {
        dmma_gemm<Tin, NT, NEG, LOWER>(M, N, K, A, lda, B, ldb, C, ldc, s);
        return 0;
    }
};
struct TcEngine {
    template <bool NT, bool NEG, bool LOWER>
    static int gemm(int M, int N, int K, const float *A, int lda, const float *B, int ldb, float *C, int ldc,
                    cudaStream_t s)
    {
        return tc::tc_gemm<NT, NEG, LOWER>(M, N, K, A, lda, B, ldb, C, ldc, s);
    }
};

// Tin = storage, Tp = panel arithmetic, E = GEMM engine.
template <typename Tin, typename Tp, class E>
int run_family(int type, int b, void *const *p, int *info, cudaStream_t s)
{
    constexpr int NBP = sizeof(Tp) == 4 ? 64 : 32;  // panel width (smem budget)
    switch (type) {
    case VS_T_MATMUL:  // C += A B                 (Fig 1)
        return E::template gemm<false, false, false>(b, b, b, (const Tin *)p[0], b, (const Tin *)p[1], b, (Tin *)p[2], b, s);
    case VS_T_GEMM_NT:  // C -= A B^T              (R5)
        return E::template gemm<true, true, false>(b, b, b, (const Tin *)p[0], b, (const Tin *)p[1], b, (Tin *)p[2], b, s);
    case VS_T_SYRK:  // C -= A A^T, lower          (R5, R7)
        return E::template gemm<true, true, true>(b, b, b, (const Tin *)p[0], b, (const Tin *)p[0], b, (Tin *)p[1], b, s);
    case VS_T_TRSM: {  // B <- B L^{-T}            (R5)
        const Tin *L = (const Tin *)p[0];
        Tin *X = (Tin *)p[1];
        for (int j0 = 0; j0 < b; j0 += NBP) {
            trsm_panel<Tin, Tp, NBP>(L + (int64_t)j0 * b + j0, b, X + j0, b, b, s);
            const int rest = b - j0 - NBP;
            if (rest > 0) {
                int r = E::template gemm<true, true, false>(b, rest, NBP, X + j0, b, L + (int64_t)(j0 + NBP) * b + j0, b,
                                                            X + j0 + NBP, b, s);
                if (r) return r;
            }
        }
        return 0;
    }
    case VS_T_POTRF: {  // A = L L^T in place      (L697-699, R9)
        Tin *A = (Tin *)p[0];
        for (int k0 = 0; k0 < b; k0 += NBP) {
            potrf_diag<Tin, Tp, NBP>(A + (int64_t)k0 * b + k0, b, k0, info, s);
            const int rest = b - k0 - NBP;
            if (rest > 0) {
                trsm_panel<Tin, Tp, NBP>(A + (int64_t)k0 * b + k0, b, A + (int64_t)(k0 + NBP) * b + k0, b, rest, s);
                Tin *P = A + (int64_t)(k0 + NBP) * b + k0;
                int r = E::template gemm<true, true, true>(rest, rest, NBP, P, b, P, b, A + (int64_t)(k0 + NBP) * b + k0 + NBP,
                                                           b, s);
                if (r) return r;
            }
        }
        return 0;
    }
    }
    return -1;
}

}  // namespace

int builtin_elem_bytes(int version) { return version >= VS_V_DFMA_F64 ? 8 : 4; }

bool builtin_supported(int type, int version, int b)
{
    if (type < 0 || type >= VS_NUM_BUILTIN_TYPES) return false;
    if (version < 0 || version >= VS_NUM_BUILTIN_VERSIONS) return false;
    if (b && (b % 64 != 0 || b < 64 || b > 4096)) return false;
    return true;
}

int launch_builtin(int type, int version, int b, void *const *p, int *info, cudaStream_t s)
{
    if (!builtin_supported(type, version, b)) return -1;
    switch (version) {
    case VS_V_SIMT_F32: return run_family<float, float, SimtEngine<float, float>>(type, b, p, info, s);
    case VS_V_TC_3XTF32: return run_family<float, float, TcEngine>(type, b, p, info, s);
    case VS_V_F64IN_F32IO: return run_family<float, double, DmmaEngine<float>>(type, b, p, info, s);
    case VS_V_DFMA_F64: return run_family<double, double, SimtEngine<double, double>>(type, b, p, info, s);
    case VS_V_DMMA_F64: return run_family<double, double, DmmaEngine<double>>(type, b, p, info, s);
    }
    return -1;
}

}  // namespace vsk
