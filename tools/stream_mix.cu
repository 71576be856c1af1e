// stream_mix.cu -- achievable HBM bandwidth for the read/write stream mixes of the hot-path
// kernels: NR input arrays summed into NW output arrays, fp64, 4096^2
// elements each (128 MiB per array, far above L2), double2 accesses, grid = SMs x 8 CTAs
// grid-striding. The copy (1R/1W) is what MEASURED_PEAKS.json reports; the SpMV is 5R/3W,
// the first fused pass 4R/3W, the last 5R/1W.
// Build: nvcc -O3 -gencode arch=compute_100a,code=sm_100a -o stream_mix tools/stream_mix.cu
#include <cstdio>
#include <cuda_runtime.h>

constexpr long long N = 4096LL * 4096LL;

template <int NR, int NW, int U>
__global__ void __launch_bounds__(256) k_mix(const double2 *const *in, double2 *const *out,
                                             long long n2) {
    // U independent elements per thread per iteration: U x NR loads in flight
    const long long stride = (long long)gridDim.x * blockDim.x;
    for (long long i0 = blockIdx.x * (long long)blockDim.x + threadIdx.x; i0 < n2;
         i0 += stride * U) {
        double2 s[U];
#pragma unroll
        for (int u = 0; u < U; ++u) s[u] = make_double2(0.0, 0.0);
#pragma unroll
        for (int r = 0; r < NR; ++r)
#pragma unroll
            for (int u = 0; u < U; ++u) {
                const long long i = i0 + u * stride;
                if (i < n2) {
                    const double2 v = __ldg(in[r] + i);
                    s[u].x += v.x;
                    s[u].y += v.y;
                }
            }
#pragma unroll
        for (int w = 0; w < NW; ++w)
#pragma unroll
            for (int u = 0; u < U; ++u) {
                const long long i = i0 + u * stride;
                if (i < n2) out[w][i] = make_double2(s[u].x + w, s[u].y);
            }
    }
}

template <int NR, int NW, int U = 1>
static void run(double2 **bufs, int nsm) {
    const double2 **din;
    double2 **dout;
    cudaMalloc(&din, sizeof(double2 *) * 8);
    cudaMalloc(&dout, sizeof(double2 *) * 8);
    cudaMemcpy(din, bufs, sizeof(double2 *) * NR, cudaMemcpyHostToDevice);
    cudaMemcpy(dout, bufs + NR, sizeof(double2 *) * NW, cudaMemcpyHostToDevice);
    const int grid = nsm * 8;
    cudaEvent_t a, b;
    cudaEventCreate(&a);
    cudaEventCreate(&b);
    float best = 1e30f;
    for (int rep = 0; rep < 12; ++rep) {
        cudaEventRecord(a);
        k_mix<NR, NW, U><<<grid, 256>>>(din, dout, N / 2);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms;
        cudaEventElapsedTime(&ms, a, b);
        if (rep >= 2 && ms < best) best = ms;
    }
    const double bytes = (double)(NR + NW) * N * 8.0;
    printf("%dR/%dW U=%d: %8.1f us  %7.1f GB/s\n", NR, NW, U, best * 1e3, bytes / (best * 1e-3) / 1e9);
    cudaFree(din);
    cudaFree(dout);
}

int main() {
    int nsm = 0;
    cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, 0);
    double2 *bufs[8];
    for (int i = 0; i < 8; ++i) {
        cudaMalloc(&bufs[i], N * sizeof(double));
        cudaMemset(bufs[i], 0, N * sizeof(double));
    }
#define ALL(U)                  \
    run<1, 1, U>(bufs, nsm);    \
    run<4, 3, U>(bufs, nsm);    \
    run<5, 3, U>(bufs, nsm);    \
    run<5, 1, U>(bufs, nsm);    \
    run<4, 2, U>(bufs, nsm);
    ALL(1) ALL(2) ALL(4)
    return 0;
}
