// probe_bulk.cu — L2 -> shared-memory bulk-copy (cp.async.bulk) throughput per SM and per chip
// as a function of copy size, bytes in flight and CTA count (one CTA per SM).
#include <cstdio>
#include <cstdint>
#include <vector>

__device__ __forceinline__ uint32_t su32(const void *p) { return (uint32_t)__cvta_generic_to_shared(p); }

__global__ void __launch_bounds__(32, 1) bulk_kernel(const uint8_t *src, size_t src_bytes, int chunk, int slots, int iters,
                                                     unsigned long long *cyc)
{
    extern __shared__ __align__(1024) uint8_t sm[];
    uint64_t *bar = (uint64_t *)(sm + (size_t)slots * chunk);
    if (threadIdx.x != 0) return;
    for (int s = 0; s < slots; s++) asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(su32(&bar[s])));
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    size_t off = ((size_t)blockIdx.x * 7919 * chunk) % (src_bytes - chunk);
    off &= ~(size_t)1023;
    const unsigned long long t0 = clock64();
    for (int i = 0; i < iters; i++) {
        const int s = i % slots;
        if (i >= slots) {
            const uint32_t par = ((i / slots) - 1) & 1;
            asm volatile("{\n\t.reg .pred P;\nW_%=:\n\tmbarrier.try_wait.parity.shared::cta.b64 P, [%0], %1;\n\t@!P bra W_%=;\n\t}" ::"r"(su32(&bar[s])), "r"(par) : "memory");
        }
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(su32(&bar[s])), "r"(chunk) : "memory");
        asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(su32(sm + (size_t)s * chunk)),
                     "l"(src + off), "r"(chunk), "r"(su32(&bar[s])) : "memory");
        off += chunk;
        if (off + chunk > src_bytes) off = 0;
    }
    for (int i = iters; i < iters + slots; i++) {
        const int s = i % slots;
        const uint32_t par = ((i / slots) - 1) & 1;
        asm volatile("{\n\t.reg .pred P;\nW_%=:\n\tmbarrier.try_wait.parity.shared::cta.b64 P, [%0], %1;\n\t@!P bra W_%=;\n\t}" ::"r"(su32(&bar[s])), "r"(par) : "memory");
    }
    cyc[blockIdx.x] = clock64() - t0;
}

int main()
{
    const size_t SRC = 64ull << 20;   // 64 MB: L2-resident after the first touch
    uint8_t *src;
    cudaMalloc(&src, SRC);
    cudaMemset(src, 1, SRC);
    unsigned long long *cyc;
    cudaMalloc(&cyc, 1024 * 8);
    cudaFuncSetAttribute(bulk_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, 220 * 1024);
    int clk;
    cudaDeviceGetAttribute(&clk, cudaDevAttrClockRate, 0);
    const int chunks[] = {4096, 16384, 32768, 65536};
    const int inflights[] = {64 << 10, 128 << 10, 192 << 10};
    const int ctas[] = {1, 16, 32, 74, 148};
    for (int ch : chunks)
        for (int inf : inflights) {
            const int slots = inf / ch;
            if (slots < 1) continue;
            for (int n : ctas) {
                const int iters = (int)((256ll << 20) / ch / 16);   // 16 MB per CTA
                cudaEvent_t e0, e1;
                cudaEventCreate(&e0);
                cudaEventCreate(&e1);
                bulk_kernel<<<n, 32, (size_t)slots * ch + 1024>>>(src, SRC, ch, slots, 64, cyc);   // warm
                cudaEventRecord(e0);
                bulk_kernel<<<n, 32, (size_t)slots * ch + 1024>>>(src, SRC, ch, slots, iters, cyc);
                cudaEventRecord(e1);
                cudaDeviceSynchronize();
                float ms;
                cudaEventElapsedTime(&ms, e0, e1);
                std::vector<unsigned long long> h(n);
                cudaMemcpy(h.data(), cyc, n * 8, cudaMemcpyDeviceToHost);
                double mc = 0;
                for (auto x : h) mc += x;
                mc /= n;
                const double bytes = (double)iters * ch;
                printf("chunk %6d inflight %4d KB ctas %3d: %.1f B/clk/SM (%.1f GB/s/SM), chip %.2f TB/s  err=%s\n", ch, inf >> 10, n,
                       bytes / mc, bytes / (ms * 1e-3) / 1e9, bytes * n / (ms * 1e-3) / 1e12, cudaGetErrorString(cudaGetLastError()));
            }
        }
    return 0;
}
