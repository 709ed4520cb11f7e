// probe_mn.cu — standalone check of the tcgen05 tf32 MN-major B encoding variants.
// nvcc -gencode arch=compute_100a,code=sm_100a -DVSK_MN_VARIANT=v -I include -o probe_v tools/probe_mn.cu
#include <cstdio>
#include <cstdlib>
#include <cmath>
#include <vector>
#include "../paper_conf_ipps_planasbal13_b200/csrc/kernels/tc_gemm.cuh"

int main()
{
    const int M = 256, N = 256, K = 128;
    std::vector<float> A(M * K), B(K * N), C(M * N, 0.f);
    for (auto &x : A) x = (float)(rand() % 17 - 8);
    for (auto &x : B) x = (float)(rand() % 17 - 8);
    float *dA, *dB, *dC;
    cudaMalloc(&dA, A.size() * 4); cudaMalloc(&dB, B.size() * 4); cudaMalloc(&dC, C.size() * 4);
    cudaMemcpy(dA, A.data(), A.size() * 4, cudaMemcpyHostToDevice);
    cudaMemcpy(dB, B.data(), B.size() * 4, cudaMemcpyHostToDevice);
    cudaMemset(dC, 0, C.size() * 4);
    vsk::tc::tc_gemm<false, false, false, true>(M, N, K, dA, K, dB, N, dC, N, 0);
    cudaError_t e = cudaDeviceSynchronize();
    cudaMemcpy(C.data(), dC, C.size() * 4, cudaMemcpyDeviceToHost);
    double maxerr = 0, maxref = 0;
    int bad = 0;
    for (int i = 0; i < M; i++)
        for (int j = 0; j < N; j++) {
            double r = 0;
            for (int k = 0; k < K; k++) r += (double)A[i * K + k] * B[k * N + j];
            maxerr = fmax(maxerr, fabs(r - C[i * N + j]));
            maxref = fmax(maxref, fabs(r));
            bad += fabs(r - C[i * N + j]) > 0.5;
        }
    printf("variant %d: err=%s maxerr=%.3g maxref=%.3g bad=%d/%d C[0]=%g C[1]=%g\n", VSK_MN_VARIANT,
           cudaGetErrorString(e), maxerr, maxref, bad, M * N, C[0], C[1]);
    return 0;
}
