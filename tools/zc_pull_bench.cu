// Ceiling of the miss path's PCIe leg: SM loads from pinned, device-mapped
// host memory ("pull", what acquire_batch does) vs a copy-engine
// cudaMemcpyAsync H2D of the same bytes. Build: nvcc -O3 -gencode
// arch=compute_100a,code=sm_100a tools/zc_pull_bench.cu -o /tmp/zc
#include <cstdio>
#include <cuda_runtime.h>

template <int U, bool CV>
__global__ void pull(const int4* __restrict__ src, int4* __restrict__ dst, size_t n16, size_t chunk16) {
  // each block copies contiguous chunks (like one page per block)
  for (size_t c0 = (size_t)blockIdx.x * chunk16; c0 < n16; c0 += (size_t)gridDim.x * chunk16) {
    const size_t end = c0 + chunk16 < n16 ? c0 + chunk16 : n16;
    for (size_t i = c0 + threadIdx.x; i < end; i += (size_t)U * blockDim.x) {
      int4 v[U];
#pragma unroll
      for (int u = 0; u < U; ++u) {
        const size_t k = i + (size_t)u * blockDim.x;
        if (k < end) v[u] = CV ? __ldcv(src + k) : src[k];
      }
#pragma unroll
      for (int u = 0; u < U; ++u) {
        const size_t k = i + (size_t)u * blockDim.x;
        if (k < end) dst[k] = v[u];
      }
    }
  }
}

int main() {
  const size_t bytes = 1ull << 30;
  void* h;
  cudaHostAlloc(&h, bytes, cudaHostAllocMapped);
  memset(h, 1, bytes);
  void* hd;
  cudaHostGetDevicePointer(&hd, h, 0);
  void* d;
  cudaMalloc(&d, bytes);
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  float ms;
  for (int r = 0; r < 3; ++r) {
    cudaEventRecord(a);
    cudaMemcpyAsync(d, h, bytes, cudaMemcpyHostToDevice);
    cudaEventRecord(b);
    cudaEventSynchronize(b);
    cudaEventElapsedTime(&ms, a, b);
  }
  printf("memcpy H2D 1 GiB: %.1f GB/s\n", bytes / ms / 1e6);
  const size_t n16 = bytes / 16;
  const size_t chunks[2] = {(2u << 20) / 16, (64u << 10) / 16};
  for (size_t ch : chunks) {
    for (int grid : {148, 296, 592, 1184}) {
      for (int threads : {256, 512}) {
        auto run = [&](auto kern, const char* name) {
          for (int r = 0; r < 2; ++r) {
            cudaEventRecord(a);
            kern<<<grid, threads>>>((const int4*)hd, (int4*)d, n16, ch);
            cudaEventRecord(b);
            cudaEventSynchronize(b);
            cudaEventElapsedTime(&ms, a, b);
          }
          printf("pull %-8s chunk=%4zuKiB grid=%4d thr=%3d: %.1f GB/s\n", name, ch * 16 >> 10, grid, threads,
                 bytes / ms / 1e6);
        };
        run(pull<4, true>, "cv,u4");
        run(pull<8, true>, "cv,u8");
        run(pull<16, false>, "ld,u16");
      }
    }
  }
  printf("%s\n", cudaGetErrorString(cudaGetLastError()));
  return 0;
}
