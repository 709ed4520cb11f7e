// builtin.cu — the built-in tile task versions (VS_T_* x VS_V_*): each version is a
// sequence of sm_100a kernels enqueued on the worker's stream.
#include "kernels.hpp"
#include "simt_chol.cuh"
#include "simt_gemm.cuh"
#include "tc_gemm.cuh"

#include "vsched.h"

namespace vsk {

namespace {

// --------------------------------------------------------------- SIMT families
// Tin = storage, Tacc = arithmetic.  simt_f32: <float,float>; f64in_f32io: <float,double>;
// dfma_f64: <double,double>.
template <typename Tin, typename Tacc>
int run_simt(int type, int b, void *const *p, int *info, cudaStream_t s)
{
    constexpr int NBP = sizeof(Tacc) == 4 ? 64 : 32;  // panel width (smem budget)
    switch (type) {
    case VS_T_MATMUL:  // C += A B
        simt_gemm<Tin, Tacc, false, false, false>(b, b, b, (const Tin *)p[0], b, (const Tin *)p[1], b, (Tin *)p[2], b, s);
        return 0;
    case VS_T_GEMM_NT:  // C -= A B^T
        simt_gemm<Tin, Tacc, true, true, false>(b, b, b, (const Tin *)p[0], b, (const Tin *)p[1], b, (Tin *)p[2], b, s);
        return 0;
    case VS_T_SYRK:  // C -= A A^T, lower
        simt_gemm<Tin, Tacc, true, true, true>(b, b, b, (const Tin *)p[0], b, (const Tin *)p[0], b, (Tin *)p[1], b, s);
        return 0;
    case VS_T_TRSM: {  // B <- B L^{-T}
        const Tin *L = (const Tin *)p[0];
        Tin *X = (Tin *)p[1];
        for (int j0 = 0; j0 < b; j0 += NBP) {
            trsm_panel<Tin, Tacc, NBP>(L + (int64_t)j0 * b + j0, b, X + j0, b, b, s);
            const int rest = b - j0 - NBP;
            if (rest > 0)
                simt_gemm<Tin, Tacc, true, true, false>(b, rest, NBP, X + j0, b, L + (int64_t)(j0 + NBP) * b + j0, b,
                                                        X + j0 + NBP, b, s);
        }
        return 0;
    }
    case VS_T_POTRF: {  // A = L L^T in place
        Tin *A = (Tin *)p[0];
        for (int k0 = 0; k0 < b; k0 += NBP) {
            potrf_diag<Tin, Tacc, NBP>(A + (int64_t)k0 * b + k0, b, k0, info, s);
            const int rest = b - k0 - NBP;
            if (rest > 0) {
                trsm_panel<Tin, Tacc, NBP>(A + (int64_t)k0 * b + k0, b, A + (int64_t)(k0 + NBP) * b + k0, b, rest, s);
                Tin *P = A + (int64_t)(k0 + NBP) * b + k0;
                simt_gemm<Tin, Tacc, true, true, true>(rest, rest, NBP, P, b, P, b, A + (int64_t)(k0 + NBP) * b + k0 + NBP, b, s);
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
    if (b && (b % 64 != 0 || b < 64 || b > 4096)) return false;
    switch (version) {
    case VS_V_SIMT_F32:
    case VS_V_F64IN_F32IO:
    case VS_V_DFMA_F64:
        return true;
    case VS_V_TC_3XTF32:
        return tc_available(type);
    default:
        return false;
    }
}

int launch_builtin(int type, int version, int b, void *const *p, int *info, cudaStream_t s)
{
    if (!builtin_supported(type, version, b)) return -1;
    switch (version) {
    case VS_V_SIMT_F32: return run_simt<float, float>(type, b, p, info, s);
    case VS_V_F64IN_F32IO: return run_simt<float, double>(type, b, p, info, s);
    case VS_V_DFMA_F64: return run_simt<double, double>(type, b, p, info, s);
    case VS_V_TC_3XTF32: return run_tc(type, b, p, info, s);
    }
    return -1;
}

}  // namespace vsk
