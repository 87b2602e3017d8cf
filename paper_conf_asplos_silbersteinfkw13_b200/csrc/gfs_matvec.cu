// gfs_matvec.cu — out-of-core fp32 matrix-vector product over GPUfs
// (§5.1.4, Fig. 8).
//
// "employing gmmap to read the data in the kernel, gftruncate to truncate the
// output file at the start, gwrite to write the output, and finally gfsync to
// synchronize the data". A is a row-major little-endian fp32
// file (rows x cols), x a cols-long fp32 file, y a rows-long fp32 output file.
//   k_mv_trunc  gopen(y, O_GWRONCE), gftruncate(y, 0)
//   k_mv_x      gread x into device memory (L2-resident afterwards)
//   k_mv_rows   block b owns rows [b*R/G, (b+1)*R/G): each row is consumed
//               through gmmap one mapped prefix at a time (<= one cache page,
//               P:L426-428) straight out of the frame; products are
//               accumulated in fp64 per thread, reduced across the block, and
//               rounded to fp32 (R16); the block gwrites its slice
//               of y once
//   k_mv_sync   gopen(y, O_GWRONCE), gfsync, gclose
// The matrix pages stream through the cache (files larger than the cache are
// the point of Fig. 8); the sampled LRU evicts them behind the sweep.
#include <cuda_runtime.h>
#include <errno.h>
#include <stdint.h>
#include <stdio.h>
#include <string.h>

#include "gpufs.h"
#include "gpufs_device.cuh"
#include "gfs_launch.h"

#define GFS_API extern "C" __attribute__((visibility("default")))

using namespace gfs;

namespace {

__device__ __forceinline__ void mv_err(int64_t* err, int64_t r) {
  if (r < 0 && err) atomicMin((long long*)err, (long long)r);
}

__global__ void k_mv_trunc(const __grid_constant__ gfs_ctx cv_, const char* y_path, int64_t* err) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  const int fd = gopen(c, y_path, GFS_O_GWRONCE);
  if (fd < 0) {
    if (threadIdx.x == 0) mv_err(err, fd);
    return;
  }
  const int r = gftruncate(c, fd, 0);
  if (threadIdx.x == 0) mv_err(err, r);
  // no gclose: y stays open until k_mv_sync, so the row blocks' gopen/gclose
  // never bounce it through the closed-file table (a write-once re-open starts
  // a new incarnation)
}

__global__ void k_mv_x(const __grid_constant__ gfs_ctx cv_, const char* x_path, uint64_t cols, float* x, int64_t* err) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  const int fd = gopen(c, x_path, GFS_O_RDONLY);
  if (fd < 0) {
    if (threadIdx.x == 0 && blockIdx.x == 0) mv_err(err, fd);
    return;
  }
  const uint64_t bytes = cols * 4, chunk = 1u << 20;
  for (uint64_t o = (uint64_t)blockIdx.x * chunk; o < bytes; o += (uint64_t)gridDim.x * chunk) {
    const uint64_t n = bytes - o < chunk ? bytes - o : chunk;
    const int64_t r = gread(c, fd, o, n, (uint8_t*)x + o);
    if (threadIdx.x == 0 && r != (int64_t)n) mv_err(err, r < 0 ? r : -EIO);
  }
  gclose(c, fd);
}

__device__ __forceinline__ double block_sum(double v, double* red) {
  for (int o = 16; o; o >>= 1) v += __shfl_xor_sync(0xFFFFFFFFu, v, o);
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5, nw = (blockDim.x + 31) >> 5;
  __syncthreads();
  if (lane == 0) red[wid] = v;
  __syncthreads();
  double s = 0.0;
  if (threadIdx.x == 0)
    for (int q = 0; q < nw; ++q) s += red[q];
  return s;  // valid in thread 0
}

// Rows [row0, row0 + nrows) of A; y (file and d_y) holds those rows only.
__global__ void __launch_bounds__(256) k_mv_rows(const __grid_constant__ gfs_ctx cv_, const char* a_path, const char* y_path,
                                                  uint64_t row0, uint64_t nrows, uint64_t cols, uint64_t per,
                                                  const float* x, float* y_dev, int64_t* err) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  extern __shared__ __align__(16) float ys[];  // this block's y slice
  __shared__ double red[32];
  const int tid = threadIdx.x, nthr = blockDim.x;
  const uint64_t r0 = row0 + blockIdx.x * per, r1 = r0 + per < row0 + nrows ? r0 + per : row0 + nrows;
  if (r0 >= r1) return;
  const int fa = gopen(c, a_path, GFS_O_RDONLY);
  if (fa < 0) {
    if (tid == 0) mv_err(err, fa);
    return;
  }
  const uint64_t rowb = cols * 4;
  bool ok = true;
  for (uint64_t r = r0; r < r1 && ok; ++r) {
    double acc = 0.0;
    uint64_t done = 0;  // bytes of row r consumed
    while (done < rowb) {
      uint64_t m = 0;
      const uint8_t* p = (const uint8_t*)gmmap(c, nullptr, rowb - done, 0, 0, fa, r * rowb + done, &m);
      if (!p || m == 0 || (m & 3) || (done & 3)) {
        if (tid == 0) mv_err(err, p ? -EINVAL : -EIO);
        if (p) gmunmap(c, (void*)p, m);
        ok = false;
        break;
      }
      const float* a = (const float*)p;
      const float* xs = x + (done >> 2);
      const uint64_t n = m >> 2;
      if ((((uintptr_t)a | (uintptr_t)xs) & 15) == 0) {
        const uint64_t n4 = n >> 2;
        for (uint64_t i = tid; i < n4; i += nthr) {
          const float4 av = __ldcg((const float4*)a + i);  // frame bytes: bypass L1 (refilled frames)
          const float4 xv = __ldg((const float4*)xs + i);
          acc += (double)av.x * xv.x + (double)av.y * xv.y + (double)av.z * xv.z + (double)av.w * xv.w;
        }
        for (uint64_t i = (n4 << 2) + tid; i < n; i += nthr) acc += (double)__ldcg(a + i) * __ldg(xs + i);
      } else {
        for (uint64_t i = tid; i < n; i += nthr) acc += (double)__ldcg(a + i) * __ldg(xs + i);
      }
      gmunmap(c, (void*)p, m);
      done += m;
    }
    if (!ok) break;
    const double s = block_sum(acc, red);
    if (tid == 0) ys[r - r0] = (float)s;
  }
  gclose(c, fa);
  __syncthreads();
  if (!ok) return;
  if (y_dev)
    for (uint64_t i = tid; i < r1 - r0; i += nthr) y_dev[r0 - row0 + i] = ys[i];
  const int fy = gopen(c, y_path, GFS_O_GWRONCE);
  if (fy < 0) {
    if (tid == 0) mv_err(err, fy);
    return;
  }
  const int64_t w = gwrite(c, fy, (r0 - row0) * 4, (r1 - r0) * 4, ys);
  if (tid == 0 && w != (int64_t)((r1 - r0) * 4)) mv_err(err, w < 0 ? w : -EIO);
  gclose(c, fy);
}

__global__ void k_mv_sync(const __grid_constant__ gfs_ctx cv_, const char* y_path, int64_t* err) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  const int fd = gopen(c, y_path, GFS_O_GWRONCE);
  if (fd < 0) {
    if (threadIdx.x == 0) mv_err(err, fd);
    return;
  }
  const int r = gfsync(c, fd);
  if (threadIdx.x == 0) mv_err(err, r);
  gclose(c, fd);
  gclose(c, fd);  // the reference k_mv_trunc kept
}

}  // namespace

GFS_API int gfs_matvec_rows(gfs_handle* h, void* stream, const char* a_path, const char* x_path, const char* y_path,
                            uint64_t rows, uint64_t cols, uint64_t row0, uint64_t nrows, float* d_x, float* d_y,
                            int64_t* d_err, uint32_t grid, uint32_t block) {
  if (!h || !a_path || !x_path || !y_path || !d_x || !d_err || rows == 0 || cols == 0 || grid == 0 ||
      block == 0 || block > 256 || (block & 31) || nrows == 0 || row0 >= rows || nrows > rows - row0)
    return -EINVAL;
  // Rows per block: ceil(nrows / grid), rounded up to whole cache pages when a
  // page holds whole rows, so no page is shared by two blocks (a shared page
  // makes one block wait for the other's fill, or fetch it a second time after
  // an eviction); blocks past the last row return at once.
  uint64_t per = (nrows + grid - 1) / grid;
  {
    const uint64_t P = gfs_launch::ctx_val(h).page_size, rowb = cols * 4;
    if (rowb <= P && P % rowb == 0 && (row0 * rowb) % P == 0) {
      const uint64_t rpp = P / rowb;
      per = (per + rpp - 1) / rpp * rpp;
    }
  }
  if (per * 4 > 160 * 1024) return -EINVAL;  // y slice must fit in shared memory: use more blocks
  cudaStream_t s = (cudaStream_t)stream;
  gfs_launch::ArgStage as(h, s);
  const char* ps[3] = {a_path, x_path, y_path};
  if (const int e = as.stage(ps, 3)) return e;
  const gfs_ctx c = gfs_launch::ctx_val(h);
  const char* da = as.str(0);
  const char* dx = as.str(1);
  const char* dy = as.str(2);
  const size_t smem = (size_t)per * 4;
  if (smem > 48 * 1024) cudaFuncSetAttribute(k_mv_rows, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  cudaMemsetAsync(d_err, 0, 8, s);
  k_mv_trunc<<<1, 128, 0, s>>>(c, dy, d_err);
  k_mv_x<<<64, 256, 0, s>>>(c, dx, cols, d_x, d_err);
  k_mv_rows<<<grid, block, smem, s>>>(c, da, dy, row0, nrows, cols, per, d_x, d_y, d_err);
  k_mv_sync<<<1, 256, 0, s>>>(c, dy, d_err);
  const cudaError_t e = cudaGetLastError();
  if (e != cudaSuccess) fprintf(stderr, "gfs_matvec: launch failed: %s\n", cudaGetErrorString(e));
  return e == cudaSuccess ? 0 : -EIO;
}

GFS_API int gfs_matvec(gfs_handle* h, void* stream, const char* a_path, const char* x_path, const char* y_path,
                       uint64_t rows, uint64_t cols, float* d_x, float* d_y, int64_t* d_err, uint32_t grid,
                       uint32_t block) {
  return gfs_matvec_rows(h, stream, a_path, x_path, y_path, rows, cols, 0, rows, d_x, d_y, d_err, grid, block);
}
