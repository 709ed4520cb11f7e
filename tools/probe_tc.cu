// probe_tc.cu — standalone check of tc_gemm over (NT, NEG, LOWER, B_MN) combinations.
#include <cstdio>
#include <cstdlib>
#include <cmath>
#include <vector>
#include "../paper_conf_ipps_planasbal13_b200/csrc/kernels/tc_gemm.cuh"

template <bool NT, bool NEG, bool LOWER, bool BMN>
void run(int M, int N, int K)
{
    std::vector<float> A(M * K), B(K * N), C(M * N), C0(M * N);
    for (auto &x : A) x = (float)(rand() % 17 - 8);
    for (auto &x : B) x = (float)(rand() % 17 - 8);
    for (auto &x : C0) x = (float)(rand() % 17 - 8);
    float *dA, *dB, *dC;
    cudaMalloc(&dA, A.size() * 4); cudaMalloc(&dB, B.size() * 4); cudaMalloc(&dC, C.size() * 4);
    cudaMemcpy(dA, A.data(), A.size() * 4, cudaMemcpyHostToDevice);
    cudaMemcpy(dB, B.data(), B.size() * 4, cudaMemcpyHostToDevice);
    cudaMemcpy(dC, C0.data(), C.size() * 4, cudaMemcpyHostToDevice);
    int ldb = NT ? K : N;
    vsk::tc::tc_gemm<NT, NEG, LOWER, BMN>(M, N, K, dA, K, dB, ldb, dC, N, 0);
    cudaError_t e = cudaDeviceSynchronize();
    cudaMemcpy(C.data(), dC, C.size() * 4, cudaMemcpyDeviceToHost);
    int bad = 0, unchanged = 0;
    for (int i = 0; i < M; i++)
        for (int j = 0; j < N; j++) {
            double r = 0;
            for (int k = 0; k < K; k++) r += (double)A[i * K + k] * (NT ? B[j * K + k] : B[k * N + j]);
            double ref = C0[i * N + j] + (NEG ? -r : r);
            if (LOWER && j > i) ref = C0[i * N + j];
            bad += fabs(ref - C[i * N + j]) > 0.5;
            unchanged += C[i * N + j] == C0[i * N + j];
        }
    printf("NT=%d NEG=%d LOWER=%d BMN=%d M=%d N=%d K=%d: %s bad=%d unchanged=%d of %d\n", NT, NEG, LOWER, BMN, M, N, K,
           cudaGetErrorString(e), bad, unchanged, M * N);
    cudaFree(dA); cudaFree(dB); cudaFree(dC);
}

int main()
{
    run<true, true, false, false>(256, 256, 128);
    run<true, false, false, false>(256, 256, 128);
    run<false, true, false, false>(256, 256, 128);
    run<false, false, false, false>(256, 256, 128);
    run<false, false, false, true>(256, 256, 128);
    run<false, true, false, true>(256, 256, 128);
    run<true, true, true, false>(256, 256, 128);
    run<false, false, false, false>(1024, 1024, 1024);
    return 0;
}
