// gen.cu — device input generator, bit-identical to vsgen.uniform_idx / vsgen.spd
// (the same counter-based function implemented on each side; DESIGN.md input recipe).
// Holds no arithmetic of the method.
#include "kernels.hpp"

#include <cmath>

namespace vsk {

__device__ __forceinline__ uint64_t splitmix64(uint64_t x)
{
    uint64_t z = x + 0x9E3779B97F4A7C15ull;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
    return z ^ (z >> 31);
}

__device__ __forceinline__ double u01(uint64_t seed, uint64_t idx)
{
    const uint64_t z = splitmix64((seed << 40) | idx);
    return (double)(z >> 40) * 0x1p-23 - 1.0;
}

// element e of the output buffer -> global (r, c)
__device__ __forceinline__ void coords(int64_t e, int64_t cols, int tile_b, int64_t &r, int64_t &c)
{
    if (!tile_b) {
        r = e / cols;
        c = e % cols;
        return;
    }
    const int64_t tb2 = (int64_t)tile_b * tile_b;
    const int64_t t = e / tb2, w = e % tb2;
    const int64_t ntc = cols / tile_b;
    r = (t / ntc) * tile_b + w / tile_b;
    c = (t % ntc) * tile_b + w % tile_b;
}

template <typename T>
__global__ void gen_uniform_kernel(uint64_t seed, int64_t rows, int64_t cols, int tile_b, T *out)
{
    const int64_t total = rows * cols;
    for (int64_t e = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; e < total; e += (int64_t)gridDim.x * blockDim.x) {
        int64_t r, c;
        coords(e, cols, tile_b, r, c);
        out[e] = (T)u01(seed, (uint64_t)(r * cols + c));
    }
}

template <typename T>
__global__ void gen_spd_kernel(uint64_t seed, int64_t n, int tile_b, double alpha, T *out)
{
    const int64_t total = n * n;
    for (int64_t e = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; e < total; e += (int64_t)gridDim.x * blockDim.x) {
        int64_t r, c;
        coords(e, n, tile_b, r, c);
        const int64_t hi = r > c ? r : c, lo = r > c ? c : r;
        double v = u01(seed, (uint64_t)(hi * n + lo));
        if (r == c) v = v + alpha;
        out[e] = (T)v;
    }
}

int gen_uniform(uint64_t seed, int64_t rows, int64_t cols, int dtype, int tile_b, void *out, cudaStream_t s)
{
    const int grid = 148 * 16;
    count_launch();
    if (dtype == 0) gen_uniform_kernel<float><<<grid, 256, 0, s>>>(seed, rows, cols, tile_b, (float *)out);
    else if (dtype == 1) gen_uniform_kernel<double><<<grid, 256, 0, s>>>(seed, rows, cols, tile_b, (double *)out);
    else return -1;
    return 0;
}

int gen_spd(uint64_t seed, int64_t n, int dtype, int tile_b, void *out, cudaStream_t s)
{
    const double alpha = n >= 256 ? 2.5 * std::sqrt((double)n) : (double)n;  // reading R8
    const int grid = 148 * 16;
    count_launch();
    if (dtype == 0) gen_spd_kernel<float><<<grid, 256, 0, s>>>(seed, n, tile_b, alpha, (float *)out);
    else if (dtype == 1) gen_spd_kernel<double><<<grid, 256, 0, s>>>(seed, n, tile_b, alpha, (double *)out);
    else return -1;
    return 0;
}

}  // namespace vsk

namespace vsk {

// One b x b tile (global tile coordinates ti, tj) of a rows x cols uniform matrix, or of
// the n x n SPD matrix (spd != 0): same values as the whole-matrix generators.
template <typename T>
__global__ void gen_tile_kernel(uint64_t seed, int64_t cols, int b, int64_t ti, int64_t tj, int spd, double alpha,
                                T *out)
{
    const int64_t total = (int64_t)b * b;
    for (int64_t e = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; e < total; e += (int64_t)gridDim.x * blockDim.x) {
        const int64_t r = ti * b + e / b, c = tj * b + e % b;
        double v;
        if (spd) {
            const int64_t hi = r > c ? r : c, lo = r > c ? c : r;
            v = u01(seed, (uint64_t)(hi * cols + lo));
            if (r == c) v = v + alpha;
        } else {
            v = u01(seed, (uint64_t)(r * cols + c));
        }
        out[e] = (T)v;
    }
}

int gen_tile(uint64_t seed, int64_t rows, int64_t cols, int dtype, int b, int64_t ti, int64_t tj, int spd, void *out,
             cudaStream_t s)
{
    (void)rows;
    const double alpha = cols >= 256 ? 2.5 * std::sqrt((double)cols) : (double)cols;  // reading R8 (n = cols)
    const int grid = 148 * 4;
    count_launch();
    if (dtype == 0) gen_tile_kernel<float><<<grid, 256, 0, s>>>(seed, cols, b, ti, tj, spd, alpha, (float *)out);
    else if (dtype == 1) gen_tile_kernel<double><<<grid, 256, 0, s>>>(seed, cols, b, ti, tj, spd, alpha, (double *)out);
    else return -1;
    return 0;
}

}  // namespace vsk
