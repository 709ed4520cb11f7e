// probe_tc.cu — standalone correctness + timing of tc_gemm over (NT, NEG, LOWER, BN).
#include <cstdio>
#include <cstdlib>
#include <cmath>
#include <vector>
#include "../paper_conf_ipps_planasbal13_b200/csrc/kernels/tc_gemm2.cuh"

template <bool NT, bool NEG, bool LOWER, int BN>
void run(int M, int N, int K, int reps = 0)
{
    std::vector<float> A((size_t)M * K), B((size_t)K * N), C((size_t)M * N), C0((size_t)M * N);
    for (auto &x : A) x = (float)(rand() % 17 - 8);
    for (auto &x : B) x = (float)(rand() % 17 - 8);
    for (auto &x : C0) x = (float)(rand() % 17 - 8);
    float *dA, *dB, *dC;
    cudaMalloc(&dA, A.size() * 4); cudaMalloc(&dB, B.size() * 4); cudaMalloc(&dC, C.size() * 4);
    cudaMemcpy(dA, A.data(), A.size() * 4, cudaMemcpyHostToDevice);
    cudaMemcpy(dB, B.data(), B.size() * 4, cudaMemcpyHostToDevice);
    cudaMemcpy(dC, C0.data(), C.size() * 4, cudaMemcpyHostToDevice);
    int ldb = NT ? K : N;
    vsk::tc2::tc_gemm2<NT, NEG, LOWER>(M, N, K, dA, K, dB, ldb, dC, N, 0);
    cudaError_t e = cudaDeviceSynchronize();
    cudaMemcpy(C.data(), dC, C.size() * 4, cudaMemcpyDeviceToHost);
    long bad = 0, unchanged = 0;
    int step = M * N > 300000 ? 61 : 1;
    for (int i = 0; i < M; i += step)
        for (int j = 0; j < N; j++) {
            double r = 0;
            for (int k = 0; k < K; k++) r += (double)A[(size_t)i * K + k] * (NT ? B[(size_t)j * K + k] : B[(size_t)k * N + j]);
            double ref = C0[(size_t)i * N + j] + (NEG ? -r : r);
            if (LOWER && j > i) ref = C0[(size_t)i * N + j];
            bad += fabs(ref - C[(size_t)i * N + j]) > 0.5;
            unchanged += C[(size_t)i * N + j] == C0[(size_t)i * N + j];
        }
    float ms = 0;
    if (reps) {
        cudaEvent_t a, b;
        cudaEventCreate(&a); cudaEventCreate(&b);
        cudaEventRecord(a);
        for (int r = 0; r < reps; r++) vsk::tc2::tc_gemm2<NT, NEG, LOWER>(M, N, K, dA, K, dB, ldb, dC, N, 0);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        cudaEventElapsedTime(&ms, a, b);
        ms /= reps;
    }
    double tf = reps ? 2.0 * M * N * K / (ms * 1e-3) / 1e12 : 0;
    printf("NT=%d NEG=%d LOWER=%d BN=%d M=%d N=%d K=%d: %s bad=%ld unchanged=%ld  %.1f us  %.1f TF alg  %.1f TF hw\n",
           NT, NEG, LOWER, BN, M, N, K, cudaGetErrorString(e), bad, unchanged, ms * 1e3, tf, 3 * tf);
    cudaFree(dA); cudaFree(dB); cudaFree(dC);
}

int main()
{
    setvbuf(stdout, NULL, _IONBF, 0);
    run<true, true, false, 256>(256, 512, 128);
    run<false, false, false, 256>(256, 512, 128);
    run<true, true, true, 256>(512, 512, 128);
    run<false, false, false, 256>(320, 320, 96);
    run<false, false, false, 256>(1024, 1024, 1024, 20);
    run<true, true, false, 256>(1024, 1024, 1024, 20);
    run<false, false, false, 256>(4096, 4096, 4096, 10);
    run<true, true, false, 256>(4096, 4096, 4096, 10);
    return 0;
}
