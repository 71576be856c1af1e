// tmem_probe.cu -- micro-benchmark: per-thread delay lines in shared memory vs in tensor
// memory (TMEM, tcgen05.st / tcgen05.ld .32x32b), as used by the fused Chebyshev passes
// (DESIGN.md §4.4). Each thread writes one double2 per "row" and reads back NR double2
// written 1..NR rows earlier. Prints bytes read per clock per SM for both.
// Build: nvcc -O3 -gencode arch=compute_100a,code=sm_100a -o tmem_probe tools/tmem_probe.cu
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

constexpr int T = 128;  // threads per CTA (one warpgroup: warp w owns TMEM lanes 32w..)
constexpr int D = 8;    // ring depth

template <int NR>
__global__ void __launch_bounds__(T) k_smem(int iters, double *out) {
    __shared__ double2 ring[D][T];
    const int tid = threadIdx.x;
    for (int d = 0; d < D; ++d) ring[d][tid] = make_double2(tid, d);
    __syncwarp();
    double2 acc = make_double2(0, 0), v = make_double2(1.0 + tid, 2.0);
#pragma unroll 1
    for (int i = 0; i < iters; ++i) {
        ring[i & (D - 1)][tid] = v;
#pragma unroll
        for (int t = 1; t <= NR; ++t) {
            const double2 x = ring[(i - t) & (D - 1)][tid];
            acc.x += x.x;
            acc.y += x.y;
        }
        v.x += 1.0;
    }
    out[blockIdx.x * T + tid] = acc.x + acc.y;
}

__device__ __forceinline__ void tst4(uint32_t a, double2 v) {
    const unsigned long long x = __double_as_longlong(v.x), y = __double_as_longlong(v.y);
    asm volatile("tcgen05.st.sync.aligned.32x32b.x4.b32 [%0], {%1, %2, %3, %4};" ::"r"(a),
                 "r"((uint32_t)x), "r"((uint32_t)(x >> 32)), "r"((uint32_t)y),
                 "r"((uint32_t)(y >> 32))
                 : "memory");
}
__device__ __forceinline__ void tld4(uint32_t a, uint32_t &r0, uint32_t &r1, uint32_t &r2,
                                     uint32_t &r3) {
    asm volatile("tcgen05.ld.sync.aligned.32x32b.x4.b32 {%0, %1, %2, %3}, [%4];"
                 : "=r"(r0), "=r"(r1), "=r"(r2), "=r"(r3)
                 : "r"(a)
                 : "memory");
}

template <int NR>
__global__ void __launch_bounds__(T) k_tmem(int iters, double *out) {
    __shared__ uint32_t base;
    const int tid = threadIdx.x, warp = tid >> 5;
    if (warp == 0) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], 32;" ::"r"(
                         (uint32_t)__cvta_generic_to_shared(&base))
                     : "memory");
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
    }
    asm volatile("tcgen05.fence::before_thread_sync;");
    __syncthreads();
    asm volatile("tcgen05.fence::after_thread_sync;");
    const uint32_t tb = base + ((uint32_t)(warp * 32) << 16);
    for (int d = 0; d < D; ++d) tst4(tb + 4 * d, make_double2(tid, d));
    asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");
    double2 acc = make_double2(0, 0), v = make_double2(1.0 + tid, 2.0);
#pragma unroll 1
    for (int i = 0; i < iters; ++i) {
        tst4(tb + 4 * (i & (D - 1)), v);
        uint32_t r[NR][4];
#pragma unroll
        for (int t = 1; t <= NR; ++t)
            tld4(tb + 4 * ((i - t) & (D - 1)), r[t - 1][0], r[t - 1][1], r[t - 1][2], r[t - 1][3]);
        asm volatile("tcgen05.wait::ld.sync.aligned;" ::: "memory");
#pragma unroll
        for (int t = 0; t < NR; ++t) {
            acc.x += __longlong_as_double(((unsigned long long)r[t][1] << 32) | r[t][0]);
            acc.y += __longlong_as_double(((unsigned long long)r[t][3] << 32) | r[t][2]);
        }
        v.x += 1.0;
        asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");
    }
    out[blockIdx.x * T + tid] = acc.x + acc.y;
    asm volatile("tcgen05.fence::before_thread_sync;");
    __syncthreads();
    if (warp == 0)
        asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, 32;" ::"r"(base));
}

template <typename K>
static void run(const char *name, K kern, int ctas_per_sm, int nr, double *out, int nsm,
                double clk_ghz) {
    const int iters = 20000;
    const int grid = nsm * ctas_per_sm;
    kern<<<grid, T>>>(100, out);
    cudaEvent_t a, b;
    cudaEventCreate(&a);
    cudaEventCreate(&b);
    cudaEventRecord(a);
    kern<<<grid, T>>>(iters, out);
    cudaEventRecord(b);
    cudaError_t e = cudaEventSynchronize(b);
    float ms = 0;
    cudaEventElapsedTime(&ms, a, b);
    if (e != cudaSuccess) {
        printf("%s: %s\n", name, cudaGetErrorString(e));
        return;
    }
    const double bytes = (double)grid * T * iters * nr * 16.0;
    const double per_sm_clk = bytes / (ms * 1e-3) / nsm / (clk_ghz * 1e9);
    printf("%-6s NR=%d ctas/SM=%d warps/SM=%2d: %8.3f ms  read %7.1f B/clk/SM  (%.0f GB/s chip)\n",
           name, nr, ctas_per_sm, ctas_per_sm * 4, ms, per_sm_clk, bytes / (ms * 1e-3) / 1e9);
}

int main() {
    int nsm = 0, khz = 0;
    cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, 0);
    cudaDeviceGetAttribute(&khz, cudaDevAttrClockRate, 0);
    const double ghz = khz * 1e-6;
    printf("SMs %d, clock %.3f GHz (max; actual may be lower)\n", nsm, ghz);
    double *out;
    cudaMalloc(&out, sizeof(double) * nsm * 16 * T);
    for (int c : {1, 2, 3, 4}) {
        run("smem", k_smem<3>, c, 3, out, nsm, ghz);
        run("tmem", k_tmem<3>, c, 3, out, nsm, ghz);
        run("smem", k_smem<6>, c, 6, out, nsm, ghz);
        run("tmem", k_tmem<6>, c, 6, out, nsm, ghz);
    }
    return 0;
}
