// probe_tcf.cu — per-CTA phase timeline of the tc_3xf16 GEMM (tc_f16.cuh built with
// -DVS_TCF_TRACE): one b x b NT task alone, then S concurrent tasks on S streams.
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -std=c++17 -DVS_TCF_TRACE -o tools/probe_tcf tools/probe_tcf.cu
#include <cstdio>
#include <cstdlib>
#include <vector>

#include "../paper_conf_ipps_planasbal13_b200/csrc/kernels/tc_f16.cuh"

using namespace vsk;

__global__ void fill(float *p, size_t n, unsigned seed)
{
    for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n; i += (size_t)gridDim.x * blockDim.x) {
        unsigned x = (unsigned)i * 2654435761u ^ seed;
        x ^= x >> 13; x *= 0x5bd1e995u; x ^= x >> 15;
        p[i] = (x & 0xFFFFFF) * (1.f / 16777216.f) * 2.f - 1.f;
    }
}

int main(int argc, char **argv)
{
    const int b = argc > 1 ? atoi(argv[1]) : 1024;
    const int S = argc > 2 ? atoi(argv[2]) : 16;
    const size_t fb = tcf::split_bytes(b, b);
    std::vector<float *> A(S), B(S), C(S);
    std::vector<void *> FA(S), FB(S);
    std::vector<cudaStream_t> st(S);
    for (int i = 0; i < S; i++) {
        cudaMalloc(&A[i], (size_t)b * b * 4); cudaMalloc(&B[i], (size_t)b * b * 4); cudaMalloc(&C[i], (size_t)b * b * 4);
        cudaMalloc(&FA[i], fb); cudaMalloc(&FB[i], fb);
        fill<<<256, 256>>>(A[i], (size_t)b * b, 1 + i); fill<<<256, 256>>>(B[i], (size_t)b * b, 100 + i);
        cudaMemset(C[i], 0, (size_t)b * b * 4);
        tcf::split_rows(A[i], b, b, b, FA[i], 0);
        tcf::split_rows(B[i], b, b, b, FB[i], 0);
        cudaStreamCreateWithFlags(&st[i], cudaStreamNonBlocking);
    }
    cudaDeviceSynchronize();
    unsigned long long *tr;
    cudaGetSymbolAddress((void **)&tr, tcf::g_tcf_trace);
    const int nct = ((b + 255) / 256) * ((b + 255) / 256);
    for (int rep = 0; rep < 3; rep++) {
        cudaMemset(tr, 0, sizeof(unsigned long long) * 1024 * 12);
        cudaEvent_t e0, e1;
        cudaEventCreate(&e0); cudaEventCreate(&e1);
        cudaEventRecord(e0, st[0]);
        tcf::tcf_gemm<true, false>(b, b, b, FA[0], FB[0], C[0], b, st[0]);
        cudaEventRecord(e1, st[0]);
        cudaDeviceSynchronize();
        float ms;
        cudaEventElapsedTime(&ms, e0, e1);
        std::vector<unsigned long long> h(1024 * 12);
        cudaMemcpy(h.data(), tr, h.size() * 8, cudaMemcpyDeviceToHost);
        unsigned long long t0 = ~0ull;
        for (int c = 0; c < nct; c++) t0 = std::min(t0, h[c * 12 + 0]);
        if (getenv("VS_TCF_PAIR") && atoi(getenv("VS_TCF_PAIR"))) {   // pair grid: x = row blocks
        }
        printf("rep %d alone: %.2f us (event)  err=%s\n", rep, ms * 1e3, cudaGetErrorString(cudaGetLastError()));
        if (rep == 2)
            for (int c = 0; c < nct; c += (nct > 8 ? nct / 8 - 1 : 1)) {
                unsigned long long *x = &h[c * 12];
                printf("  cta %3d start %6.2f alloc %6.2f full0 %6.2f fullmid %6.2f lastmma %6.2f cin %6.2f accfull %6.2f epi_end %6.2f end %6.2f | fullwait %6.2f pairwait %6.2f us\n",
                       c, (x[0] - t0) / 1e3, (x[1] - t0) / 1e3, (x[2] - t0) / 1e3, (x[3] - t0) / 1e3, x[4] ? (x[4] - t0) / 1e3 : 0.0,
                       (x[5] - t0) / 1e3, (x[6] - t0) / 1e3, (x[8] - t0) / 1e3, (x[7] - t0) / 1e3, x[9] / 1e3, x[10] / 1e3);
            }
    }
    // S concurrent tasks, 20 rounds
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0); cudaEventCreate(&e1);
    for (int w = 0; w < 10; w++) {
        const int SS = w < 2 ? 6 : w < 4 ? 8 : w < 6 ? 10 : w < 8 ? 12 : 16;
        if (SS > S) break;
        cudaEventRecord(e0, 0);
        for (int i = 0; i < SS; i++) cudaStreamWaitEvent(st[i], e0, 0);
        const int R = 20;
        for (int r = 0; r < R; r++)
            for (int i = 0; i < SS; i++) tcf::tcf_gemm<true, false>(b, b, b, FA[i], FB[i], C[i], b, st[i]);
        for (int i = 0; i < SS; i++) {
            cudaEvent_t e;
            cudaEventCreate(&e);
            cudaEventRecord(e, st[i]);
            cudaStreamWaitEvent(0, e, 0);
        }
        cudaEventRecord(e1, 0);
        cudaDeviceSynchronize();
        float ms;
        cudaEventElapsedTime(&ms, e0, e1);
        printf("%d streams: %.2f us per task, %.1f TF/s algorithmic\n", SS, ms * 1e3 / (R * SS), 2.0 * b * b * (double)b * R * SS / (ms * 1e-3) / 1e12);
    }
    return 0;
}
