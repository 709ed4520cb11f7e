// fig4_versions.cu — the Fig 4 fixture of PAPER.md (L296-345, Sec IV.A) as USER versions of
// one task, registered through vs_version_add ("implements(main_impl)"): three CUDA
// implementations of
//
//     task input([N]A) output([N]B) inout([N]C)   f(int N, float *A, float *B, float *C)
//
// with identical parameters and in/out sets (L306-308).  The paper leaves the body as "Task
// code"; the fixture's body is  B[i] = A[i] + A[i];  C[i] = fmaf(A[i], A[i], C[i])  (the same
// IEEE result in every version).  The versions differ only in how they map the work to the
// GPU, so their speeds differ, which is what the versioning scheduler learns:
//   main_impl        one thread per element
//   another_impl     float4 grid-stride loop over 4 x 148 CTAs
//   yet_another_one  a single CTA walking the whole array (deliberately slow)
// Each follows the vs_launch_fn contract of include/vsched.h: enqueue on `stream`, never
// synchronise it, touch only the task's parameters, deterministic.  N arrives as the task's
// scalar (the int N parameter of Fig 4); it is checked against the parameter sizes.
// TEST INFRASTRUCTURE: built by tests/test_gpu_api.py (nvcc -shared), not part of libvsched.
#include <cuda_runtime.h>
#include <stdint.h>
#include <string.h>

namespace {

__global__ void main_impl_kernel(int n, const float *__restrict__ A, float *__restrict__ B, float *__restrict__ C)
{
    const int i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i < n) {
        const float a = A[i];
        B[i] = a + a;
        C[i] = fmaf(a, a, C[i]);
    }
}

__global__ void another_impl_kernel(int n, const float *__restrict__ A, float *__restrict__ B, float *__restrict__ C)
{
    const int n4 = n / 4;
    for (int i = blockIdx.x * blockDim.x + threadIdx.x; i < n4; i += gridDim.x * blockDim.x) {
        const float4 a = reinterpret_cast<const float4 *>(A)[i];
        float4 c = reinterpret_cast<float4 *>(C)[i];
        reinterpret_cast<float4 *>(B)[i] = make_float4(a.x + a.x, a.y + a.y, a.z + a.z, a.w + a.w);
        c = make_float4(fmaf(a.x, a.x, c.x), fmaf(a.y, a.y, c.y), fmaf(a.z, a.z, c.z), fmaf(a.w, a.w, c.w));
        reinterpret_cast<float4 *>(C)[i] = c;
    }
    for (int i = 4 * n4 + blockIdx.x * blockDim.x + threadIdx.x; i < n; i += gridDim.x * blockDim.x) {
        const float a = A[i];
        B[i] = a + a;
        C[i] = fmaf(a, a, C[i]);
    }
}

__global__ void yet_another_one_kernel(int n, const float *__restrict__ A, float *__restrict__ B, float *__restrict__ C)
{
    for (int i = threadIdx.x; i < n; i += blockDim.x) {
        const float a = A[i];
        B[i] = a + a;
        C[i] = fmaf(a, a, C[i]);
    }
}

// parameters (A in, B out, C inout) and the scalar N; 0 if they agree
int args_of(void *const *p, const int64_t *bytes, int nargs, const void *scalars, size_t nscalar, int *n)
{
    if (nargs != 3 || nscalar != sizeof(int) || !scalars) return 1;
    memcpy(n, scalars, sizeof(int));
    for (int i = 0; i < 3; i++)
        if (!p[i] || bytes[i] != (int64_t)*n * (int64_t)sizeof(float)) return 2;
    return 0;
}

}  // namespace

extern "C" {

int fig4_main_impl(void *const *p, const int64_t *bytes, int nargs, const void *scalars, size_t nscalar, void *stream,
                   void *user)
{
    (void)user;
    int n = 0;
    if (args_of(p, bytes, nargs, scalars, nscalar, &n)) return 1;
    main_impl_kernel<<<(n + 255) / 256, 256, 0, (cudaStream_t)stream>>>(n, (const float *)p[0], (float *)p[1], (float *)p[2]);
    return cudaGetLastError() == cudaSuccess ? 0 : 3;
}

int fig4_another_impl(void *const *p, const int64_t *bytes, int nargs, const void *scalars, size_t nscalar,
                      void *stream, void *user)
{
    (void)user;
    int n = 0;
    if (args_of(p, bytes, nargs, scalars, nscalar, &n)) return 1;
    another_impl_kernel<<<4 * 148, 256, 0, (cudaStream_t)stream>>>(n, (const float *)p[0], (float *)p[1], (float *)p[2]);
    return cudaGetLastError() == cudaSuccess ? 0 : 3;
}

int fig4_yet_another_one(void *const *p, const int64_t *bytes, int nargs, const void *scalars, size_t nscalar,
                         void *stream, void *user)
{
    (void)user;
    int n = 0;
    if (args_of(p, bytes, nargs, scalars, nscalar, &n)) return 1;
    yet_another_one_kernel<<<1, 256, 0, (cudaStream_t)stream>>>(n, (const float *)p[0], (float *)p[1], (float *)p[2]);
    return cudaGetLastError() == cudaSuccess ? 0 : 3;
}

// a version that violates nothing but reports failure: the runtime must surface it
int fig4_failing(void *const *p, const int64_t *bytes, int nargs, const void *scalars, size_t nscalar, void *stream,
                 void *user)
{
    (void)p, (void)bytes, (void)nargs, (void)scalars, (void)nscalar, (void)stream, (void)user;
    return 7;
}

}  // extern "C"
