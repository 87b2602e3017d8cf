// gfs_launch.h — internal helpers shared by the kernel launchers (not part of
// the C ABI): per-handle staging of string arguments (paths) in device memory.
#pragma once

#include <cuda_runtime.h>

#include "gpufs.h"

#define GFS_ARG_SLOT_BYTES (4 * GFS_MAX_PATH)  /* up to 4 strings per launch */

extern "C" int gfs_internal_args(gfs_handle* h, cudaStream_t s, const char* const* strs, int n, char** d_out);
extern "C" void gfs_internal_args_done(gfs_handle* h, int slot, cudaStream_t s);
extern "C" int gfs_internal_device(gfs_handle* h);
// The host copy of the handle's context (what gfs_device_ctx points to on the
// device, kept in step with it): launchers pass it BY VALUE as a
// __grid_constant__ kernel parameter, so the kernel reads the context's
// fields from the constant bank instead of L1/L2. Launchers copy it without a
// lock: gfs_export / gfs_attach_peer (the only calls that change it after
// gfs_init) must not run concurrently with launches on the same handle from
// other threads (as before, when kernels read the device copy they update).
extern "C" const gfs_ctx* gfs_internal_host_ctx(gfs_handle* h);

namespace gfs_launch {
// The context a kernel takes by value (zeros for kernels launched without a
// handle, e.g. the raw baselines, which never read it).
inline gfs_ctx ctx_val(gfs_handle* h) {
  gfs_ctx v{};
  if (const gfs_ctx* p = h ? gfs_internal_host_ctx(h) : nullptr) v = *p;
  return v;
}


// Scope of one launcher call: makes the handle's device current, stages the
// strings in a slot of the handle's ring, and — when the launcher returns,
// i.e. after its last kernel is enqueued — records the slot's reuse event on
// the stream and restores the caller's device.
struct ArgStage {
  gfs_handle* h;
  cudaStream_t s;
  int slot = -1;
  int prev_dev = -1;
  char* d = nullptr;
  ArgStage(gfs_handle* h_, cudaStream_t s_) : h(h_), s(s_) {
    if (h && cudaGetDevice(&prev_dev) == cudaSuccess) cudaSetDevice(gfs_internal_device(h));
  }
  // 0 or -errno
  int stage(const char* const* strs, int n) {
    if (!h) return -EINVAL;
    const int k = gfs_internal_args(h, s, strs, n, &d);
    if (k < 0) return k;
    slot = k;
    return 0;
  }
  const char* str(int i) const { return d ? d + (size_t)i * GFS_MAX_PATH : nullptr; }
  ~ArgStage() {
    if (slot >= 0) gfs_internal_args_done(h, slot, s);
    if (h && prev_dev >= 0) cudaSetDevice(prev_dev);
  }
  ArgStage(const ArgStage&) = delete;
  ArgStage& operator=(const ArgStage&) = delete;
};

}  // namespace gfs_launch
