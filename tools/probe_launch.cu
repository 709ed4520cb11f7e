// Host cost of the CUDA runtime calls the executor makes per task (B200, one thread):
// kernel launches with 64 B / 512 B / 2 KB / 4 KB parameter blocks, cudaEventRecord,
// cudaStreamWaitEvent, cudaSetDevice, cudaEventQuery.  Kernels are empty; 8 streams
// round-robin as in the runtime.
//   nvcc -gencode arch=compute_100a,code=sm_100a -O2 -o /tmp/probe_launch tools/probe_launch.cu
#include <chrono>
#include <cstdio>
#include <cuda_runtime.h>

template <int BYTES>
struct P {
    char b[BYTES];
};
template <int BYTES>
__global__ void k(const __grid_constant__ P<BYTES> p)
{
    if (threadIdx.x == 1024) printf("%d", p.b[0]);
}

static double now_us()
{
    return std::chrono::duration<double, std::micro>(std::chrono::steady_clock::now().time_since_epoch()).count();
}

template <int BYTES>
void launch_cost(cudaStream_t *st, int nst, int n)
{
    P<BYTES> p{};
    for (int i = 0; i < 100; i++) k<BYTES><<<16, 128, 0, st[i % nst]>>>(p);
    cudaDeviceSynchronize();
    double t0 = now_us();
    for (int i = 0; i < n; i++) k<BYTES><<<16, 128, 0, st[i % nst]>>>(p);
    double t1 = now_us();
    cudaDeviceSynchronize();
    printf("launch %5d B params: %.2f us/launch\n", BYTES, (t1 - t0) / n);
}

int main()
{
    const int NS = 8, N = 20000;
    cudaStream_t st[NS];
    for (int i = 0; i < NS; i++) cudaStreamCreateWithFlags(&st[i], cudaStreamNonBlocking);
    launch_cost<64>(st, NS, N);
    launch_cost<512>(st, NS, N);
    launch_cost<2112>(st, NS, N);
    launch_cost<4000>(st, NS, N);
    cudaEvent_t ev[64];
    for (int i = 0; i < 64; i++) cudaEventCreateWithFlags(&ev[i], cudaEventDisableTiming);
    double t0 = now_us();
    for (int i = 0; i < N; i++) cudaEventRecord(ev[i % 64], st[i % NS]);
    double t1 = now_us();
    cudaDeviceSynchronize();
    printf("cudaEventRecord: %.2f us\n", (t1 - t0) / N);
    t0 = now_us();
    for (int i = 0; i < N; i++) cudaStreamWaitEvent(st[(i + 1) % NS], ev[i % 64], 0);
    t1 = now_us();
    cudaDeviceSynchronize();
    printf("cudaStreamWaitEvent: %.2f us\n", (t1 - t0) / N);
    t0 = now_us();
    for (int i = 0; i < N; i++) cudaSetDevice(0);
    t1 = now_us();
    printf("cudaSetDevice: %.3f us\n", (t1 - t0) / N);
    t0 = now_us();
    for (int i = 0; i < N; i++) (void)cudaEventQuery(ev[i % 64]);
    t1 = now_us();
    printf("cudaEventQuery: %.3f us\n", (t1 - t0) / N);
    // launch + record interleaved (what flush_group does per group)
    P<2112> p{};
    t0 = now_us();
    for (int i = 0; i < N; i++) {
        k<2112><<<16, 128, 0, st[i % NS]>>>(p);
        cudaEventRecord(ev[i % 64], st[i % NS]);
    }
    t1 = now_us();
    cudaDeviceSynchronize();
    printf("launch(2 KB)+record: %.2f us\n", (t1 - t0) / N);
    return 0;
}
