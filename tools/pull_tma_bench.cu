// Host->device pull mechanisms over PCIe for the miss path: (ce) cudaMemcpyAsync,
// (ld) SM 16-byte loads of mapped pinned memory (k_link_pull), (tma) cp.async.bulk
// of mapped pinned memory into shared memory, then a bulk store to global, 2 stages
// per block. Usage: pull_tma_bench [MiB] [chunk KiB] [blocks per SM]
#include <cuda_runtime.h>
#include <stdio.h>
#include <stdint.h>
#include <stdlib.h>
__device__ __forceinline__ uint32_t su32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__global__ void k_ld(const int4* src, int4* dst, uint64_t n16) {
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n16; i += stride) dst[i] = __ldcv(src + i);
}
__global__ void k_tma(const uint8_t* src, uint8_t* dst, uint64_t n, uint32_t chunk) {
  extern __shared__ __align__(128) uint8_t sm[];
  __shared__ __align__(8) uint64_t mb[2];
  if (threadIdx.x == 0) {
    for (int i = 0; i < 2; ++i) asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(su32(&mb[i])));
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  if (threadIdx.x != 0) return;
  uint32_t ph[2] = {0, 0};
  const uint64_t nch = n / chunk;
  int k = 0;
  uint64_t pend[2] = {~0ull, ~0ull};
  for (uint64_t c = blockIdx.x; c < nch + 2 * gridDim.x; c += gridDim.x, k ^= 1) {
    if (pend[k] != ~0ull) {  // wait for the load into buffer k, store it
      asm volatile("{ .reg .pred P; W: mbarrier.try_wait.parity.shared::cta.b64 P, [%0], %1; @!P bra W; }" ::"r"(su32(&mb[k])), "r"(ph[k]) : "memory");
      ph[k] ^= 1;
      asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;" ::"l"(dst + pend[k] * chunk), "r"(su32(sm + k * chunk)), "r"(chunk) : "memory");
      asm volatile("cp.async.bulk.commit_group;" ::: "memory");
      asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory");  // smem buffer free again
      pend[k] = ~0ull;
    }
    if (c < nch) {
      asm volatile("{ .reg .b64 st; mbarrier.arrive.expect_tx.shared::cta.b64 st, [%0], %1; }" ::"r"(su32(&mb[k])), "r"(chunk) : "memory");
      asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(su32(sm + k * chunk)), "l"(src + c * chunk), "r"(chunk), "r"(su32(&mb[k])) : "memory");
      pend[k] = c;
    }
  }
  asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
}
int main(int argc, char** argv) {
  const uint64_t n = (uint64_t)(argc > 1 ? atoi(argv[1]) : 256) << 20;
  const uint32_t chunk = (uint32_t)(argc > 2 ? atoi(argv[2]) : 32) << 10;
  const int per_sm = argc > 3 ? atoi(argv[3]) : 2;
  uint8_t *h, *hd, *d;
  cudaHostAlloc((void**)&h, n, cudaHostAllocMapped);
  for (uint64_t i = 0; i < n; ++i) h[i] = (uint8_t)(i * 7);
  cudaHostGetDevicePointer((void**)&hd, h, 0);
  cudaMalloc((void**)&d, n);
  int nsm;
  cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, 0);
  cudaFuncSetAttribute(k_tma, cudaFuncAttributeMaxDynamicSharedMemorySize, 2 * chunk);
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  float ms;
  double bce = 0, bld = 0, btma = 0;
  for (int r = 0; r < 10; ++r) {
    cudaEventRecord(e0); cudaMemcpyAsync(d, h, n, cudaMemcpyHostToDevice); cudaEventRecord(e1); cudaEventSynchronize(e1);
    cudaEventElapsedTime(&ms, e0, e1); bce = fmax(bce, n / (ms * 1e6));
    cudaEventRecord(e0); k_ld<<<nsm * 8, 256>>>((const int4*)hd, (int4*)d, n / 16); cudaEventRecord(e1); cudaEventSynchronize(e1);
    cudaEventElapsedTime(&ms, e0, e1); bld = fmax(bld, n / (ms * 1e6));
    cudaMemset(d, 0, n);
    cudaEventRecord(e0); k_tma<<<nsm * per_sm, 32, 2 * chunk>>>(hd, d, n, chunk); cudaEventRecord(e1); cudaEventSynchronize(e1);
    cudaEventElapsedTime(&ms, e0, e1); btma = fmax(btma, n / (ms * 1e6));
  }
  uint8_t* chk = (uint8_t*)malloc(n);
  cudaMemcpy(chk, d, n, cudaMemcpyDeviceToHost);
  uint64_t bad = 0;
  for (uint64_t i = 0; i < n; ++i) bad += chk[i] != (uint8_t)(i * 7);
  printf("%llu MiB, chunk %u KiB, %d blocks/SM: copy engine %.1f GB/s, SM loads %.1f GB/s, TMA %.1f GB/s (bad bytes %llu) err %s\n",
         (unsigned long long)(n >> 20), chunk >> 10, per_sm, bce, bld, btma, (unsigned long long)bad, cudaGetErrorString(cudaGetLastError()));
  return 0;
}
