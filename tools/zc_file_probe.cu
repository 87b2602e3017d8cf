// Feasibility probe for a zero-copy miss path: register a tmpfs file's shared
// mapping with CUDA (cudaHostRegister) and let SMs pull file pages straight
// from the page cache (no daemon memcpy into staging). Reports the
// registration time and the pull bandwidth vs pinned cudaMemcpyAsync.
// Build: nvcc -O3 -gencode arch=compute_100a,code=sm_100a tools/zc_file_probe.cu -o /tmp/zcf
#include <cstdio>
#include <cstdlib>
#include <chrono>
#include <fcntl.h>
#include <sys/mman.h>
#include <sys/stat.h>
#include <unistd.h>
#include <cuda_runtime.h>

__global__ void pull(const int4* __restrict__ src, int4* __restrict__ dst, size_t n16, size_t chunk16,
                     unsigned long long* sum) {
  unsigned long long s = 0;
  for (size_t c0 = (size_t)blockIdx.x * chunk16; c0 < n16; c0 += (size_t)gridDim.x * chunk16) {
    const size_t end = c0 + chunk16 < n16 ? c0 + chunk16 : n16;
    for (size_t i = c0 + threadIdx.x; i < end; i += 4 * (size_t)blockDim.x) {
      int4 v[4];
#pragma unroll
      for (int u = 0; u < 4; ++u) {
        const size_t k = i + (size_t)u * blockDim.x;
        if (k < end) v[u] = __ldcv(src + k);
      }
#pragma unroll
      for (int u = 0; u < 4; ++u) {
        const size_t k = i + (size_t)u * blockDim.x;
        if (k < end) {
          dst[k] = v[u];
          s += (unsigned)v[u].x;
        }
      }
    }
  }
  atomicAdd(sum, s);
}

int main(int argc, char** argv) {
  const char* path = argc > 1 ? argv[1] : "/dev/shm/zc_probe.bin";
  const size_t bytes = (argc > 2 ? strtoull(argv[2], 0, 0) : 1ull) << 30;
  int fd = open(path, O_RDWR | O_CREAT, 0644);
  if (fd < 0 || ftruncate(fd, bytes) != 0) { perror("file"); return 1; }
  {  // fill (page cache resident)
    char* w = (char*)malloc(1 << 20);
    for (int i = 0; i < (1 << 20); ++i) w[i] = (char)(i * 131 + 7);
    for (size_t o = 0; o < bytes; o += 1 << 20)
      if (pwrite(fd, w, 1 << 20, o) != (1 << 20)) { perror("pwrite"); return 1; }
    free(w);
  }
  void* map = mmap(nullptr, bytes, getenv("ZC_RO") ? PROT_READ : (PROT_READ | PROT_WRITE), MAP_SHARED, fd, 0);
  if (map == MAP_FAILED) { perror("mmap"); return 1; }
  auto t0 = std::chrono::steady_clock::now();
  cudaError_t e = cudaHostRegister(map, bytes, cudaHostRegisterMapped | cudaHostRegisterReadOnly);
  auto t1 = std::chrono::steady_clock::now();
  printf("cudaHostRegister(%zu MiB shared tmpfs mapping, read-only): %s in %.1f ms\n", bytes >> 20,
         cudaGetErrorString(e), std::chrono::duration<double, std::milli>(t1 - t0).count());
  if (e != cudaSuccess) {
    e = cudaHostRegister(map, bytes, cudaHostRegisterMapped);
    printf("  retry without ReadOnly: %s\n", cudaGetErrorString(e));
    if (e != cudaSuccess) return 0;
  }
  void* dptr = nullptr;
  cudaHostGetDevicePointer(&dptr, map, 0);
  int4* dst;
  unsigned long long* sum;
  cudaMalloc(&dst, bytes);
  cudaMalloc(&sum, 8);
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  for (int grid : {148, 296, 592}) {
    for (size_t chunk : {(size_t)2 << 20, (size_t)256 << 10}) {
      float best = 1e9;
      for (int r = 0; r < 5; ++r) {
        cudaEventRecord(a);
        pull<<<grid, 256>>>((const int4*)dptr, dst, bytes / 16, chunk / 16, sum);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms;
        cudaEventElapsedTime(&ms, a, b);
        if (ms < best) best = ms;
      }
      printf("zero-copy pull from the file mapping: grid %d, %zu KiB per block: %.1f GB/s\n", grid, chunk >> 10,
             bytes / (best * 1e-3) / 1e9);
    }
  }
  void* pinned;
  cudaHostAlloc(&pinned, bytes, cudaHostAllocDefault);
  float best = 1e9;
  for (int r = 0; r < 5; ++r) {
    cudaEventRecord(a);
    cudaMemcpyAsync(dst, pinned, bytes, cudaMemcpyHostToDevice);
    cudaEventRecord(b);
    cudaEventSynchronize(b);
    float ms;
    cudaEventElapsedTime(&ms, a, b);
    if (ms < best) best = ms;
  }
  printf("pinned cudaMemcpyAsync H2D: %.1f GB/s\n", bytes / (best * 1e-3) / 1e9);
  auto t2 = std::chrono::steady_clock::now();
  cudaHostUnregister(map);
  auto t3 = std::chrono::steady_clock::now();
  printf("cudaHostUnregister: %.1f ms\n", std::chrono::duration<double, std::milli>(t3 - t2).count());
  unlink(path);
  return 0;
}
