// gfs_kernels.cu — kernels built on the device API (gpufs_device.cuh) and the
// extern "C" launchers declared in include/gpufs.h.
//
//   k_init_metadata   pframe/counter initialisation at gfs_init
//   k_gread_calls     parity harness: per-block gopen + gread/gmmap calls
//   k_seqread         C2 / K1 sequential sweep + position checksum
//   k_randread        K4 cache-hit reads into shared memory and
//                     its raw-memory baseline with the same access pattern
//   k_gwrite_calls    gwrite harness (O_GWRONCE)
//   k_fileop          gfsync / gftruncate / gfstat / gopen+gclose
#include <cuda_runtime.h>

#include <algorithm>
#include <errno.h>
#include <stdint.h>
#include <string.h>

#include "gpufs.h"
#include "gpufs_device.cuh"
#include "gfs_launch.h"

#define GFS_API extern "C" __attribute__((visibility("default")))

using namespace gfs;

namespace {

__global__ void k_init_metadata(gfs_ctx c) {
  const size_t stride = (size_t)gridDim.x * blockDim.x;
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < c.nframes; i += stride) {
    c.f_state[i] = (uint64_t)GFS_ST_EVICTING;  // never-used frames are handed out by fresh_next only
    c.f_tag[i] = GFS_TAG_NONE;
    c.f_file[i] = 0xFFFFFFFFu;
    c.f_valid[i] = 0;
    c.f_lo[i] = GFS_DIRTY_NONE;
    c.f_hi[i] = 0;
    c.f_written[i] = 0;
    c.f_stamp[i] = 0;
    c.f_hv[i] = 0;
    c.f_pristine[i] = 0;
    c.f_pf[i] = 0;
  }
  if (blockIdx.x == 0 && threadIdx.x == 0) {
    *c.fresh_next = 0;
    *c.hand = 0;
    *c.node_next = 1;  // node 0 is the null node
    *c.node_free_top = 0;
    *c.node_lock = 0;
    *c.uid_next = 1;
  }
}

// Position-weighted checksum of `n` bytes at `p` holding file bytes starting at
// file offset `foff` (8-byte aligned): sum_j w_j * (2j + 1), j global word index.
__device__ __forceinline__ uint64_t checksum_words(const uint8_t* p, uint64_t foff, uint64_t n, int tid,
                                                   int nthr, bool cg) {
  uint64_t s = 0;
  const uint64_t j0 = foff >> 3;
  const uint64_t nw = n >> 3;
  if (((uintptr_t)p & 15) == 0) {
    const uint64_t nv = nw >> 1;
    const ulonglong2* p2 = (const ulonglong2*)p;
    for (uint64_t i = tid; i < nv; i += nthr) {
      ulonglong2 v = cg ? __ldcg(p2 + i) : p2[i];
      const uint64_t j = j0 + 2 * i;
      s += v.x * (2 * j + 1) + v.y * (2 * j + 3);
    }
    if ((nw & 1) && tid == 0) {
      const uint64_t* p1 = (const uint64_t*)p;
      s += (cg ? __ldcg(p1 + nw - 1) : p1[nw - 1]) * (2 * (j0 + nw - 1) + 1);
    }
  } else {
    for (uint64_t i = tid; i < nw; i += nthr) {
      uint64_t v = 0;
      for (int b = 0; b < 8; ++b) v |= (uint64_t)p[8 * i + b] << (8 * b);
      s += v * (2 * (j0 + i) + 1);
    }
  }
  if (tid == 0 && (n & 7)) {  // ragged tail: missing bytes count as zero
    uint64_t v = 0;
    for (uint64_t b = 0; b < (n & 7); ++b) v |= (uint64_t)p[8 * nw + b] << (8 * b);
    s += v * (2 * (j0 + nw) + 1);
  }
  return s;
}

__device__ __forceinline__ uint64_t warp_sum(uint64_t v) {
  for (int o = 16; o; o >>= 1) v += __shfl_xor_sync(0xFFFFFFFFu, v, o);
  return v;
}

__device__ __forceinline__ void note_err(int64_t* d_err, int64_t r) {
  if (r < 0 && d_err) atomicMin((long long*)d_err, (long long)r);
}

__global__ void k_gread_calls(const __grid_constant__ gfs_ctx cv_, const char* path, int mode, uint32_t ncalls, const uint64_t* off,
                              const uint64_t* len, const uint64_t* dstoff, uint8_t* dst, int64_t* ret,
                              uint32_t smem_bytes) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  extern __shared__ __align__(16) uint8_t smem[];
  const int tid = threadIdx.x;
  const int fd = gopen(c, path, mode >> 8);  // open flags ride in the high bits (O_RDONLY or O_RDWR)
  mode &= 0xFF;
  for (uint32_t i = blockIdx.x; i < ncalls; i += gridDim.x) {
    int64_t r;
    if (fd < 0) {
      r = fd;
    } else if (mode == 0) {
      r = gread(c, fd, off[i], len[i], dst + dstoff[i]);
    } else if (mode == 1) {
      uint64_t m = 0;
      uint8_t* p = (uint8_t*)gmmap(c, nullptr, len[i], 0, 0, fd, off[i], &m);
      if (p) {
        // user copy out of the mapped page (frames are read with .cg loads)
        detail::block_copy_from_frame(dst + dstoff[i], p, m, tid, blockDim.x);
        __syncthreads();
        gmunmap(c, p, m);
        r = (int64_t)m;
      } else {
        r = 0;
      }
    } else {
      // mode 2: shared buffer at its aligned base; mode 3: at off % 16, so the
      // destination is co-aligned with the file offset (TMA middle + edges)
      const uint32_t sh = mode == 3 ? (uint32_t)(off[i] & 15) : 0u;
      if (len[i] + sh > smem_bytes) {
        r = -EINVAL;  // destination would overflow the shared buffer
      } else {
        r = gread(c, fd, off[i], len[i], smem + sh);
        if (r > 0)
          for (int64_t k = tid; k < r; k += blockDim.x) dst[dstoff[i] + k] = smem[sh + k];
        __syncthreads();
      }
    }
    if (tid == 0) ret[i] = r;
  }
  if (fd >= 0) gclose(c, fd);
}

// Warp-collective variant of the parity harness (gopen_warp / gread_warp /
// gclose_warp): warp w of the grid issues calls w, w + nwarps, ...
// mode 4: into global memory; mode 5: into the warp's shared buffer
// (smem_bytes per warp) at off % 16, then copied out.
__global__ void k_gread_calls_warp(const __grid_constant__ gfs_ctx cv_, const char* path, int mode, uint32_t ncalls,
                                   const uint64_t* off, const uint64_t* len, const uint64_t* dstoff, uint8_t* dst,
                                   int64_t* ret, uint32_t smem_bytes) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  extern __shared__ __align__(16) uint8_t smem[];
  const int lane = threadIdx.x & 31, wib = threadIdx.x >> 5;
  const uint32_t gw = blockIdx.x * (blockDim.x >> 5) + wib, nw = gridDim.x * (blockDim.x >> 5);
  uint8_t* wbuf = smem + (size_t)wib * smem_bytes;
  const int fd = gopen_warp(c, path, GFS_O_RDONLY);
  for (uint32_t i = gw; i < ncalls; i += nw) {
    int64_t r;
    if (fd < 0) {
      r = fd;
    } else if (mode == 4) {
      r = gread_warp(c, fd, off[i], len[i], dst + dstoff[i]);
    } else {
      const uint32_t sh = (uint32_t)(off[i] & 15);
      if (len[i] + sh > smem_bytes) {
        r = -EINVAL;
      } else {
        r = gread_warp(c, fd, off[i], len[i], wbuf + sh);
        for (int64_t k = lane; k < r; k += 32) dst[dstoff[i] + k] = wbuf[sh + k];
        __syncwarp();
      }
    }
    if (lane == 0) ret[i] = r;
  }
  if (fd >= 0) gclose_warp(c, fd);
}

__global__ void __launch_bounds__(256, 4) k_seqread(const __grid_constant__ gfs_ctx cv_, const char* path, uint64_t file_off, uint64_t total, uint64_t chunk,
                          int use_mmap, uint8_t* scratch, uint64_t* sum, int64_t* err) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  const int tid = threadIdx.x, nthr = blockDim.x;
  const int fd = gopen(c, path, GFS_O_RDONLY);
  if (fd < 0) {
    if (tid == 0) note_err(err, fd);
    return;
  }
  const uint64_t nchunks = (total + chunk - 1) / chunk;
  const uint64_t per = (nchunks + gridDim.x - 1) / gridDim.x;
  const uint64_t c0 = blockIdx.x * per, c1 = c0 + per < nchunks ? c0 + per : nchunks;
  uint64_t s = 0;
  uint8_t* buf = scratch + (size_t)blockIdx.x * chunk;
  for (uint64_t k = c0; k < c1; ++k) {
    const uint64_t o = file_off + k * chunk;
    const uint64_t want = (k + 1) * chunk <= total ? chunk : total - k * chunk;
    if (use_mmap == 2) {  // copy only: gread into the full-size destination at the file offset (cache-hit
                          // gread -> global: 2 HBM bytes per byte, no consumer pass)
      const int64_t r = gread(c, fd, o, want, scratch + (o - file_off));
      if (r < 0) {
        if (tid == 0) note_err(err, r);
        break;
      }
    } else if (!use_mmap) {
      const int64_t r = gread(c, fd, o, want, buf);
      if (r < 0) {
        if (tid == 0) note_err(err, r);
        break;
      }
      s += checksum_words(buf, o, (uint64_t)r, tid, nthr, false);
    } else {
      uint64_t done = 0;
      while (done < want) {  // gmmap maps at most one page: loop over the prefix
        uint64_t m = 0;
        const uint8_t* p = (const uint8_t*)gmmap(c, nullptr, want - done, 0, 0, fd, o + done, &m);
        if (!p || m == 0) {
          if (tid == 0) note_err(err, -EIO);
          break;
        }
        s += checksum_words(p, o + done, m, tid, nthr, true);
        __syncthreads();
        gmunmap(c, (void*)p, m);
        done += m;
      }
    }
  }
  s = warp_sum(s);
  if ((tid & 31) == 0) atomicAdd((unsigned long long*)sum, (unsigned long long)s);
  gclose(c, fd);
}

template <bool kHint>
__global__ void __launch_bounds__(256, 4) k_randread(const __grid_constant__ gfs_ctx cv, const char* path, int raw,
                                                     const uint8_t* rawp, uint32_t chunk, uint32_t calls,
                                                     const uint64_t* offs, uint64_t* sum, int64_t* err) {
  const gfs_ctx* c = &cv;  // the context by value: its fields come from the constant bank
  extern __shared__ __align__(16) uint8_t smem[];
  const int tid = threadIdx.x, nthr = blockDim.x;
  int fd = 0;
  raw = raw == 1;
  if (!raw) {
    fd = gopen(c, path, GFS_O_RDONLY);
    if (fd < 0) {
      if (tid == 0) note_err(err, fd);
      return;
    }
  }
  uint64_t s = 0;
  const uint64_t* my = offs + (size_t)blockIdx.x * calls;
  // raw baseline: the same copy without GPUfs — TMA bulk copy like gread's
  // shared-memory path, so the comparison isolates the cache's cost
  __shared__ uint64_t raw_mbar;
  if (raw) {
    if (tid == 0) detail::mbar_init(&raw_mbar);
    __syncthreads();
  }
  uint32_t ph = 0;
  for (uint32_t i = 0; i < calls; ++i) {
    const uint64_t o = my[i];
    int64_t r;
    if (raw) {
      __syncthreads();
      if (tid == 0) {
        asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
        detail::mbar_expect_tx(&raw_mbar, chunk);
        detail::tma_load(smem, rawp + o, chunk, &raw_mbar);
      }
      detail::mbar_wait(&raw_mbar, ph);
      ph ^= 1u;
      __syncthreads();
      r = chunk;
    } else {
      if constexpr (kHint) r = gread_hint(c, fd, o, chunk, smem, i + 1 < calls ? my[i + 1] : ~0ull);
      else r = gread(c, fd, o, chunk, smem);
      if (r < 0) {
        if (tid == 0) note_err(err, r);
        break;
      }
    }
    s += checksum_words(smem, o, (uint64_t)r, tid, nthr, false);
  }
  s = warp_sum(s);
  if ((tid & 31) == 0) atomicAdd((unsigned long long*)sum, (unsigned long long)s);
  if (!raw) gclose(c, fd);
}

// K4 with the warp-collective API (the paper's design point):
// every warp issues its own gread_warp calls into its own chunk of shared
// memory (warp w takes calls w, w + nwarps, ...), so one warp's lookup never
// stalls the block's other warps at a barrier. raw: the same per-warp TMA
// copies without GPUfs.
__global__ void __launch_bounds__(256) k_randread_warp(const __grid_constant__ gfs_ctx cv_, const char* path, int raw,
                                                       const uint8_t* rawp, uint32_t chunk, uint32_t calls,
                                                       const uint64_t* offs, uint64_t* sum, int64_t* err) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  extern __shared__ __align__(16) uint8_t smem[];
  __shared__ uint64_t raw_mbar[GFS_WARP_API_MAX_WARPS];
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5, nw = blockDim.x >> 5;
  uint8_t* buf = smem + (size_t)wid * chunk;
  int fd = 0;
  if (!raw) {
    fd = gopen_warp(c, path, GFS_O_RDONLY);
    if (fd < 0) {
      if (lane == 0) note_err(err, fd);
      return;
    }
  } else {
    if (lane == 0) detail::mbar_init(&raw_mbar[wid]);
    __syncwarp();
  }
  uint64_t s = 0;
  uint32_t ph = 0;
  const uint64_t* my = offs + (size_t)blockIdx.x * calls;
  for (uint32_t i = wid; i < calls; i += nw) {
    const uint64_t o = my[i];
    int64_t r;
    if (raw) {
      __syncwarp();
      if (lane == 0) {
        asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
        detail::mbar_expect_tx(&raw_mbar[wid], chunk);
        detail::tma_load(buf, rawp + o, chunk, &raw_mbar[wid]);
      }
      detail::mbar_wait(&raw_mbar[wid], ph);
      ph ^= 1u;
      r = chunk;
    } else {
      r = gread_warp(c, fd, o, chunk, buf);
      if (r < 0) {
        if (lane == 0) note_err(err, r);
        break;
      }
    }
    s += checksum_words(buf, o, (uint64_t)r, lane, 32, false);
  }
  s = warp_sum(s);
  if (lane == 0) atomicAdd((unsigned long long*)sum, (unsigned long long)s);
  if (!raw) gclose_warp(c, fd);
}

// K4 with the split-phase lane-parallel gread (NEXT-2): warp 0 issues the
// block's next `depth` calls (one lane each: lookups and TMA copies in flight)
// into one half of a double buffer while the whole block checksums the other
// half, so a call's page-table walk and copy overlap the previous calls'
// consumption. raw: the same schedule with plain TMA copies of d_raw.
__global__ void __launch_bounds__(256) k_randread_async(const __grid_constant__ gfs_ctx cv_, const char* path, int raw,
                                                        const uint8_t* rawp, uint32_t chunk, uint32_t calls,
                                                        uint32_t depth, const uint64_t* offs, uint64_t* sum,
                                                        int64_t* err) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  extern __shared__ __align__(16) uint8_t smem[];
  __shared__ uint64_t raw_mbar;
  const int tid = threadIdx.x, nthr = blockDim.x, lane = tid & 31, wid = tid >> 5;
  int fd = 0;
  if (!raw) {
    fd = gopen(c, path, GFS_O_RDONLY);  // block-collective; the warp calls below use it
    if (fd < 0) {
      if (tid == 0) note_err(err, fd);
      return;
    }
  } else if (tid == 0) {
    detail::mbar_init(&raw_mbar);
  }
  __syncthreads();
  const uint64_t* my = offs + (size_t)blockIdx.x * calls;
  GreadLaneTicket tk{0, -1, -1, 0, 0};
  uint32_t raw_ph = 0;
  // issue calls [base, base + depth) into half h (warp 0)
  auto issue = [&](uint32_t base, uint32_t h) {
    const uint32_t i = base + (uint32_t)lane;
    const bool a = (uint32_t)lane < depth && i < calls;
    uint8_t* dst = smem + ((size_t)h * depth + (a ? lane : 0)) * chunk;
    if (!raw) {
      tk = gread_lanes_issue(c, a ? fd : -1, a ? my[i] : 0, a ? chunk : 0, dst);
    } else {
      const uint32_t n = min(depth, calls - base);
      if (lane == 0) {
        asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
        detail::mbar_expect_tx(&raw_mbar, n * chunk);
      }
      __syncwarp();
      if (a) detail::tma_load(dst, rawp + my[i], chunk, &raw_mbar);
    }
  };
  auto wait = [&]() {
    if (!raw) {
      const int64_t r = gread_lanes_wait(c, tk);
      if (r < 0) note_err(err, r);
    } else {
      detail::mbar_wait(&raw_mbar, raw_ph);
      raw_ph ^= 1u;
    }
  };
  if (wid == 0) issue(0, 0);
  uint64_t s = 0;
  for (uint32_t base = 0, h = 0; base < calls; base += depth, h ^= 1u) {
    if (wid == 0) wait();  // half h holds calls [base, base + depth)
    __syncthreads();
    if (wid == 0 && base + depth < calls) issue(base + depth, h ^ 1u);
    const uint32_t n = min(depth, calls - base);
    for (uint32_t q = 0; q < n; ++q)
      s += checksum_words(smem + ((size_t)h * depth + q) * chunk, my[base + q], chunk, tid, nthr, false);
    __syncthreads();  // half h is free for the issue two rounds on
  }
  s = warp_sum(s);
  if (lane == 0) atomicAdd((unsigned long long*)sum, (unsigned long long)s);
  if (!raw) gclose(c, fd);
}

__global__ void k_gwrite_calls(const __grid_constant__ gfs_ctx cv_, const char* path, uint32_t ncalls, const uint64_t* off,
                               const uint64_t* len, const uint64_t* srcoff, const uint8_t* src, int64_t* ret,
                               int flags) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  const int fd = gopen(c, path, flags);
  for (uint32_t i = blockIdx.x; i < ncalls; i += gridDim.x) {
    int64_t r = fd < 0 ? fd : gwrite(c, fd, off[i], len[i], src + srcoff[i]);
    if (threadIdx.x == 0) ret[i] = r;
  }
  if (fd >= 0) gclose(c, fd);
}

// Writable-mapping harness (O_RDWR, Tab.1 gmsync): block i maps
// [off[i], off[i] + len[i]) with GFS_PROT_WRITE, stores src bytes through the
// pointer, optionally gmsync()s the page, and gmunmap()s. ret[i] = bytes
// mapped (the prefix) or -errno.
__global__ void k_mmap_write(const __grid_constant__ gfs_ctx cv_, const char* path, uint32_t ncalls, const uint64_t* off,
                             const uint64_t* len, const uint64_t* srcoff, const uint8_t* src, int64_t* ret,
                             int do_msync) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  const int fd = gopen(c, path, GFS_O_RDWR);
  for (uint32_t i = blockIdx.x; i < ncalls; i += gridDim.x) {
    int64_t r = fd;
    if (fd >= 0) {
      uint64_t m = 0;
      uint8_t* p = (uint8_t*)gmmap(c, nullptr, len[i], GFS_PROT_WRITE, 0, fd, off[i], &m);
      if (!p) {
        r = m ? -EIO : (int64_t)-EBADF;
      } else {
        for (uint64_t k = threadIdx.x; k < m; k += blockDim.x) p[k] = src[srcoff[i] + k];
        __threadfence();
        __syncthreads();
        r = (int64_t)m;
        if (do_msync) {
          const int e = gmsync(c, p, m, 0);
          if (e < 0) r = e;
        }
        gmunmap(c, p, m);
      }
    }
    if (threadIdx.x == 0) ret[i] = r;
  }
  if (fd >= 0) gclose(c, fd);
}

// C5 write side: every block gopen()s the (pinned, O_GWRONCE) file, gwrite()s
// its contiguous share of [0, total) from `src` in `chunk`-byte calls, gclose()s.
__global__ void k_seqwrite(const __grid_constant__ gfs_ctx cv_, const char* path, uint64_t total, uint64_t chunk, const uint8_t* src,
                           int64_t* err) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  const int fd = gopen(c, path, GFS_O_GWRONCE);
  if (fd < 0) {
    if (threadIdx.x == 0) note_err(err, fd);
    return;
  }
  const uint64_t nchunks = (total + chunk - 1) / chunk;
  const uint64_t per = (nchunks + gridDim.x - 1) / gridDim.x;
  const uint64_t c0 = blockIdx.x * per, c1 = c0 + per < nchunks ? c0 + per : nchunks;
  for (uint64_t k = c0; k < c1; ++k) {
    const uint64_t o = k * chunk, n = o + chunk <= total ? chunk : total - o;
    const int64_t r = gwrite(c, fd, o, n, src + o);
    if (r != (int64_t)n) {
      if (threadIdx.x == 0) note_err(err, r < 0 ? r : -EIO);
      break;
    }
  }
  gclose(c, fd);
}

// gfsync by every block of the grid: blocks claim dirty pages with a CAS, so
// concurrent callers split the write-back between them (each waits for its own).
// allow_busy: -EBUSY (a page claimed by a concurrent gfsync of this grid) is
// not an error here; a strict single-block pass follows and catches the rest.
__global__ void k_fsync_from_pin(const __grid_constant__ gfs_ctx cv_, const int64_t* pinned_fd, int64_t* err, int allow_busy) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  const int64_t fd = *pinned_fd;
  if (fd < 0) {
    if (threadIdx.x == 0 && blockIdx.x == 0) note_err(err, fd);
    return;
  }
  const int r = gfsync(c, (int)fd);
  if (threadIdx.x == 0 && r < 0 && !(allow_busy && r == -EBUSY)) note_err(err, r);
}

__global__ void k_unpin(const __grid_constant__ gfs_ctx cv_, const int64_t* pinned_fd, int64_t* err) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  const int64_t fd = *pinned_fd;
  if (fd < 0) return;
  const int r = gclose(c, (int)fd);
  if (threadIdx.x == 0 && r < 0) note_err(err, r);
}

__global__ void k_fileop(const __grid_constant__ gfs_ctx cv_, const char* path, int flags, int op, uint64_t arg, int64_t* ret) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  if (op == 6) {  // gfsync from every block of the grid (the pages split by claim), then a strict pass
    const int fd = gopen(c, path, flags);
    int r = fd;
    if (fd >= 0) {
      r = gfsync(c, fd);
      if (arg == 0 && r == -EBUSY) r = 0;  // a page another block of this grid was syncing
      const int cr = gclose(c, fd);
      if (r >= 0 && cr < 0) r = cr;
    }
    if (threadIdx.x == 0 && r < 0) atomicMin((long long*)ret, (long long)r);
    return;
  }
  if (op == 5) {  // unpin: drop a reference taken by op 4
    const int64_t r = gclose(c, (int)arg);
    if (threadIdx.x == 0) *ret = r;
    return;
  }
  const int fd = gopen(c, path, flags);
  int64_t r = fd;
  if (fd >= 0) {
    if (op == 0) r = gfsync(c, fd);
    else if (op == 1) r = gftruncate(c, fd, arg);
    else if (op == 2) r = gfstat_size(c, fd);
    else r = fd;
    if (op != 4) {  // op 4 = pin: keep the file open across launches
      const int cr = gclose(c, fd);
      if (r >= 0 && cr < 0) r = cr;
    }
  }
  if (threadIdx.x == 0) *ret = r;
}

int launch_err(cudaError_t e) { return e == cudaSuccess ? 0 : -EIO; }

}  // namespace

extern "C" int gfs_internal_init_metadata(gfs_ctx* hctx, cudaStream_t s) {
  k_init_metadata<<<1024, 256, 0, s>>>(*hctx);
  return launch_err(cudaGetLastError());
}

GFS_API int gfs_run_gread(gfs_handle* h, void* stream, const char* path, int mode, uint32_t ncalls,
                          const uint64_t* d_off, const uint64_t* d_len, const uint64_t* d_dstoff, uint8_t* d_dst,
                          int64_t* d_ret, uint32_t grid, uint32_t block, uint32_t smem_bytes) {
  if (!h || grid == 0 || block == 0 || block > 1024 || mode < 0 || (mode & 0xFF) > 5) return -EINVAL;
  if ((mode >> 8) != (int)GFS_O_RDONLY && (mode >> 8) != (int)GFS_O_RDWR) return -EINVAL;
  if ((mode & 0xFF) >= 4 && (mode >> 8)) return -EINVAL;  // warp harness: read-only opens
  if ((mode & 0xFF) >= 4 && ((block & 31) || block > 32 * GFS_WARP_API_MAX_WARPS)) return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  gfs_launch::ArgStage as(h, s);
  if (const int e = as.stage(&path, 1)) return e;
  const char* dp = as.str(0);
  if (mode >= 4 && mode <= 5) {
    const uint32_t dyn = mode == 5 ? smem_bytes * (block / 32) : 0;
    if (dyn > 200 * 1024) return -EINVAL;
    if (dyn > 48 * 1024)
      cudaFuncSetAttribute(k_gread_calls_warp, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)dyn);
    k_gread_calls_warp<<<grid, block, dyn, s>>>(gfs_launch::ctx_val(h), dp, mode, ncalls, d_off, d_len, d_dstoff, d_dst,
                                                d_ret, smem_bytes);
    return launch_err(cudaGetLastError());
  }
  if ((mode & 0xFF) >= 2 && smem_bytes > 48 * 1024)
    cudaFuncSetAttribute(k_gread_calls, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem_bytes);
  k_gread_calls<<<grid, block, (mode & 0xFF) >= 2 ? smem_bytes : 0, s>>>(gfs_launch::ctx_val(h), dp, mode, ncalls, d_off, d_len,
                                                                d_dstoff, d_dst, d_ret, smem_bytes);
  return launch_err(cudaGetLastError());
}

GFS_API int gfs_run_seqread(gfs_handle* h, void* stream, const char* path, uint64_t file_off, uint64_t total,
                            uint64_t chunk, int use_mmap, uint8_t* d_scratch, uint64_t* d_sum, int64_t* d_err,
                            uint32_t grid, uint32_t block) {
  if (!h || grid == 0 || block == 0 || block > 1024 || chunk == 0 || (chunk & 7) || (file_off & 7)) return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  gfs_launch::ArgStage as(h, s);
  if (const int e = as.stage(&path, 1)) return e;
  const char* dp = as.str(0);
  k_seqread<<<grid, block, 0, s>>>(gfs_launch::ctx_val(h), dp, file_off, total, chunk, use_mmap, d_scratch, d_sum, d_err);
  return launch_err(cudaGetLastError());
}

GFS_API int gfs_run_randread(gfs_handle* h, void* stream, const char* path, int raw, const uint8_t* d_raw,
                             uint32_t chunk, uint32_t calls_per_block, const uint64_t* d_off, uint64_t* d_sum,
                             int64_t* d_err, uint32_t grid, uint32_t block) {
  if (raw < 0 || raw > 2 || (raw != 1 && !h) || (raw == 1 && !d_raw) || grid == 0 || block == 0 || chunk == 0 ||
      (chunk & 15) || chunk > 200 * 1024)
    return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  gfs_launch::ArgStage as(raw == 1 ? nullptr : h, s);
  if (raw != 1)
    if (const int e = as.stage(&path, 1)) return e;
  const char* dp = raw == 1 ? nullptr : as.str(0);
  auto kern = raw == 2 ? k_randread<true> : k_randread<false>;
  if (chunk > 48 * 1024) cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)chunk);
  gfs_ctx cv{};
  if (raw != 1) cv = *gfs_internal_host_ctx(h);
  kern<<<grid, block, chunk, s>>>(cv, dp, raw, d_raw, chunk, calls_per_block, d_off, d_sum, d_err);
  return launch_err(cudaGetLastError());
}

GFS_API int gfs_run_randread_warp(gfs_handle* h, void* stream, const char* path, int raw, const uint8_t* d_raw,
                                  uint32_t chunk, uint32_t calls_per_block, const uint64_t* d_off, uint64_t* d_sum,
                                  int64_t* d_err, uint32_t grid, uint32_t block) {
  if ((!raw && !h) || (raw && !d_raw) || grid == 0 || block == 0 || (block & 31) ||
      block / 32 > GFS_WARP_API_MAX_WARPS || chunk == 0 || (chunk & 15) || (uint64_t)chunk * (block / 32) > 200 * 1024)
    return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  gfs_launch::ArgStage as(raw ? nullptr : h, s);
  if (!raw)
    if (const int e = as.stage(&path, 1)) return e;
  const char* dp = raw ? nullptr : as.str(0);
  const uint32_t smem = chunk * (block / 32);
  if (smem > 48 * 1024) cudaFuncSetAttribute(k_randread_warp, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  k_randread_warp<<<grid, block, smem, s>>>(gfs_launch::ctx_val(raw ? nullptr : h), dp, raw, d_raw, chunk,
                                             calls_per_block, d_off, d_sum, d_err);
  return launch_err(cudaGetLastError());
}

GFS_API int gfs_run_randread_async(gfs_handle* h, void* stream, const char* path, int raw, const uint8_t* d_raw,
                                   uint32_t chunk, uint32_t calls_per_block, uint32_t depth, const uint64_t* d_off,
                                   uint64_t* d_sum, int64_t* d_err, uint32_t grid, uint32_t block) {
  if ((!raw && !h) || (raw && !d_raw) || grid == 0 || block < 32 || block > 256 || (block & 31) || chunk == 0 ||
      (chunk & 15) || depth == 0 || depth > 32 || (uint64_t)chunk * depth * 2 > 200 * 1024)
    return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  gfs_launch::ArgStage as(raw ? nullptr : h, s);
  if (!raw)
    if (const int e = as.stage(&path, 1)) return e;
  const char* dp = raw ? nullptr : as.str(0);
  const uint32_t smem = chunk * depth * 2;
  if (smem > 48 * 1024) cudaFuncSetAttribute(k_randread_async, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  k_randread_async<<<grid, block, smem, s>>>(gfs_launch::ctx_val(raw ? nullptr : h), dp, raw, d_raw, chunk,
                                              calls_per_block, depth, d_off, d_sum, d_err);
  return launch_err(cudaGetLastError());
}

GFS_API int gfs_run_gwrite(gfs_handle* h, void* stream, const char* path, uint32_t ncalls, const uint64_t* d_off,
                           const uint64_t* d_len, const uint64_t* d_srcoff, const uint8_t* d_src, int64_t* d_ret,
                           uint32_t grid, uint32_t block, int flags) {
  if (!h || grid == 0 || block == 0 || block > 1024) return -EINVAL;
  if (flags != (int)GFS_O_GWRONCE && flags != (int)GFS_O_RDWR) return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  gfs_launch::ArgStage as(h, s);
  if (const int e = as.stage(&path, 1)) return e;
  const char* dp = as.str(0);
  k_gwrite_calls<<<grid, block, 0, s>>>(gfs_launch::ctx_val(h), dp, ncalls, d_off, d_len, d_srcoff, d_src, d_ret, flags);
  return launch_err(cudaGetLastError());
}

GFS_API int gfs_run_mmap_write(gfs_handle* h, void* stream, const char* path, uint32_t ncalls, const uint64_t* d_off,
                               const uint64_t* d_len, const uint64_t* d_srcoff, const uint8_t* d_src, int64_t* d_ret,
                               uint32_t grid, uint32_t block, int do_msync) {
  if (!h || grid == 0 || block == 0 || block > 1024) return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  gfs_launch::ArgStage as(h, s);
  if (const int e = as.stage(&path, 1)) return e;
  const char* dp = as.str(0);
  k_mmap_write<<<grid, block, 0, s>>>(gfs_launch::ctx_val(h), dp, ncalls, d_off, d_len, d_srcoff, d_src, d_ret, do_msync);
  return launch_err(cudaGetLastError());
}

GFS_API int gfs_run_seqwrite(gfs_handle* h, void* stream, const char* path, uint64_t total, uint64_t chunk,
                             const uint8_t* d_src, int64_t* d_err, int64_t* d_tmp, uint32_t grid, uint32_t block,
                             uint32_t sync_grid) {
  if (!h || !d_src || !d_err || !d_tmp || grid == 0 || block == 0 || block > 1024 || sync_grid == 0 || chunk == 0)
    return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  gfs_launch::ArgStage as(h, s);
  if (const int e = as.stage(&path, 1)) return e;
  const char* dp = as.str(0);
  const gfs_ctx c = gfs_launch::ctx_val(h);
  // pin: one open held across the launches, so the writers' gclose never
  // closes the file (a later O_GWRONCE open would start a new incarnation)
  k_fileop<<<1, 256, 0, s>>>(c, dp, GFS_O_GWRONCE, 4, 0, d_tmp);
  k_seqwrite<<<grid, block, 0, s>>>(c, dp, total, chunk, d_src, d_err);
  k_fsync_from_pin<<<sync_grid, block, 0, s>>>(c, d_tmp, d_err, sync_grid > 1);
  if (sync_grid > 1) k_fsync_from_pin<<<1, block, 0, s>>>(c, d_tmp, d_err, 0);  // every page clean now
  k_unpin<<<1, 32, 0, s>>>(c, d_tmp, d_err);
  return launch_err(cudaGetLastError());
}

GFS_API int gfs_run_fileop(gfs_handle* h, void* stream, const char* path, int flags, int op, uint64_t arg,
                           int64_t* d_ret) {
  if (!h || !d_ret) return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  gfs_launch::ArgStage as(h, s);
  if (const int e = as.stage(&path, 1)) return e;
  const char* dp = as.str(0);
  if (op == 6) {  // parallel gfsync: arg = grid; *d_ret = 0 or the most negative error
    if (arg == 0 || arg > 65535) return -EINVAL;
    cudaMemsetAsync(d_ret, 0, 8, s);
    k_fileop<<<(uint32_t)arg, 256, 0, s>>>(gfs_launch::ctx_val(h), dp, flags, 6, 0, d_ret);
    k_fileop<<<1, 256, 0, s>>>(gfs_launch::ctx_val(h), dp, flags, 6, 1, d_ret);  // strict: every page clean now
    return launch_err(cudaGetLastError());
  }
  k_fileop<<<1, 256, 0, s>>>(gfs_launch::ctx_val(h), dp, flags, op, arg, d_ret);
  return launch_err(cudaGetLastError());
}

// ------------------------------------------------------------------ link probe
// The host->device link as the miss path uses it: SMs pulling 16-byte words
// from mapped pinned host memory (__ldcv, like the staging pull), next to the
// copy engine's cudaMemcpyAsync. The roofline of the miss path is the faster.
__global__ void __launch_bounds__(256) k_link_pull(const int4* src, int4* dst, uint64_t n16) {
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n16; i += stride) dst[i] = __ldcv(src + i);
}

GFS_API int gfs_probe_h2d(void* stream, uint64_t nbytes, uint32_t reps, double* ce_gbps, double* sm_gbps) {
  if (!ce_gbps || !sm_gbps || nbytes < (1u << 20) || (nbytes & 15) || reps == 0) return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  uint8_t *h = nullptr, *hd = nullptr, *d = nullptr;
  if (cudaHostAlloc((void**)&h, nbytes, cudaHostAllocMapped | cudaHostAllocPortable) != cudaSuccess) return -ENOMEM;
  memset(h, 1, nbytes);  // first touch: the pages exist before the timed copies
  if (cudaHostGetDevicePointer((void**)&hd, h, 0) != cudaSuccess || cudaMalloc((void**)&d, nbytes) != cudaSuccess) {
    cudaFreeHost(h);
    return -ENOMEM;
  }
  int dev = 0, nsm = 148;
  cudaGetDevice(&dev);
  cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, dev);
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  double best_ce = 0, best_sm = 0;
  for (uint32_t r = 0; r < reps; ++r) {
    float ms = 0;
    cudaEventRecord(e0, s);
    cudaMemcpyAsync(d, h, nbytes, cudaMemcpyHostToDevice, s);
    cudaEventRecord(e1, s);
    cudaEventSynchronize(e1);
    cudaEventElapsedTime(&ms, e0, e1);
    if (ms > 0) best_ce = std::max(best_ce, nbytes / (ms * 1e6));
    cudaEventRecord(e0, s);
    k_link_pull<<<nsm * 8, 256, 0, s>>>((const int4*)hd, (int4*)d, nbytes / 16);
    cudaEventRecord(e1, s);
    cudaEventSynchronize(e1);
    cudaEventElapsedTime(&ms, e0, e1);
    if (ms > 0) best_sm = std::max(best_sm, nbytes / (ms * 1e6));
  }
  const cudaError_t e = cudaGetLastError();
  cudaEventDestroy(e0);
  cudaEventDestroy(e1);
  cudaFree(d);
  cudaFreeHost(h);
  *ce_gbps = best_ce;
  *sm_gbps = best_sm;
  return e == cudaSuccess ? 0 : -EIO;
}
