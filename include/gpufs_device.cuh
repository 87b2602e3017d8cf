// gpufs_device.cuh — header-only device library: the GPUfs API called from
// inside CUDA kernels (sm_100a), block-collectively.
//
// API (Table 1; semantics §3.2):
//
//   int     gopen (const gfs_ctx*, const char* path, int flags);
//   int     gclose(const gfs_ctx*, int fd);
//   int64_t gread (const gfs_ctx*, int fd, uint64_t off, uint64_t len, void* dst);
//   int64_t gwrite(const gfs_ctx*, int fd, uint64_t off, uint64_t len, const void* src);
//   int     gfsync(const gfs_ctx*, int fd);
//   void*   gmmap (const gfs_ctx*, void* addr, uint64_t len, int prot, int flags,
//                  int fd, uint64_t off, uint64_t* mapped_len);
//   int     gmunmap(const gfs_ctx*, void* addr, uint64_t len);
//   int64_t gfstat_size(const gfs_ctx*, int fd);
//   int     gftruncate(const gfs_ctx*, int fd, uint64_t size);
//
// Warp-collective variants (the paper's warp granularity):
// gopen_warp, gclose_warp, gfstat_size_warp, gread_warp, gmmap_warp,
// gmunmap_warp (same arguments and semantics, one warp instead of the block),
// and the vectored gread_lanes (one request per lane).
//
// Calling convention (§4): every thread of the threadblock calls
// the same function with the same arguments at the same point; each call is an
// implicit barrier and every thread receives the same return value. Negative
// returns are -errno. `dst`/`src` may point to global or shared memory and are
// owned by the caller. A gmmap pointer is borrowed until gmunmap. fds are
// GPU-global (an fd names a file): a block may use an fd another
// block opened while that open is held.
//
// Errors: -EBADF bad/closed fd, gread on O_GWRONCE, gwrite on O_RDONLY;
// -EINVAL bad flags; -ENOENT/-EACCES from host open; -EMFILE table full;
// -ENOMEM no evictable frame / node pool exhausted (deadlock guard);
// -EIO RPC or pread failure; -ENAMETOOLONG path >= GFS_MAX_PATH;
// -EBUSY gfsync skipped mapped/in-use dirty pages, or conflicting open mode;
// -ETIMEDOUT the host daemon did not answer within ctx->timeout_ns.
//
// Design: per-file radix tree (fanout 256) of u32 frame ids in
// HBM, looked up lock-free with (uid,page) tag validation; frame
// state word = refcount + FILLING/EVICTING/ERROR bits, changed only by atomic
// deltas. A miss installs a frame by CAS and posts an RPC on the pinned ring
// (P:L719-725); the host daemon preads into a pinned staging slot and stores a
// completion word in pinned memory; the installing BLOCK then pulls the page
// over PCIe into the frame and clears FILLING. No CUDA stream operation is on
// the miss path (a stream-ordered DMA can sit behind the running kernel in a
// shared hardware queue). Lookups never wait on another block's fill: they
// report BUSY and the block retries after filling its own pages, so blocks
// never wait on each other in a cycle. Eviction is a sampled, tiered LRU over
// 32-frame windows run in the calling thread. Tree slots are
// hints: evictors never touch tree nodes; a reader that finds a stale slot
// installs over it.
#pragma once

#include <stdint.h>
#include <errno.h>
#include "gpufs_layout.h"

namespace gfs {
namespace detail {
namespace {  // internal linkage: the header is included by several translation units

constexpr int kBusy = -10000;  // lookup result: page being filled/evicted elsewhere
constexpr int kLeafCache = 32; // per-block leaf-node cache entries

// ------------------------------------------------------------------ PTX
__device__ __forceinline__ uint64_t now_ns() {
  uint64_t t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
}
__device__ __forceinline__ uint32_t smid() {
  uint32_t s;
  asm volatile("mov.u32 %0, %%smid;" : "=r"(s));
  return s;
}
__device__ __forceinline__ uint32_t ld_acq(const uint32_t* p) {
  uint32_t v;
  asm volatile("ld.acquire.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ uint64_t ld_acq64(const uint64_t* p) {
  uint64_t v;
  asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ uint64_t ld_acq_sys64(const uint64_t* p) {
  uint64_t v;
  asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ uint32_t ld_rlx(const uint32_t* p) {
  uint32_t v;
  asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ uint64_t ld_rlx64(const uint64_t* p) {
  uint64_t v;
  asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_rel(uint32_t* p, uint32_t v) {
  asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ void st_rel64(uint64_t* p, uint64_t v) {
  asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ void st_rel_sys64(uint64_t* p, uint64_t v) {
  asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ void st_rlx(uint32_t* p, uint32_t v) {
  asm volatile("st.relaxed.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ void st_rlx64(uint64_t* p, uint64_t v) {
  asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ uint32_t atom_add_acq(uint32_t* p, uint32_t v) {
  uint32_t r;
  asm volatile("atom.acquire.gpu.global.add.u32 %0, [%1], %2;" : "=r"(r) : "l"(p), "r"(v) : "memory");
  return r;
}
__device__ __forceinline__ uint32_t atom_add_rel(uint32_t* p, uint32_t v) {
  uint32_t r;
  asm volatile("atom.release.gpu.global.add.u32 %0, [%1], %2;" : "=r"(r) : "l"(p), "r"(v) : "memory");
  return r;
}
__device__ __forceinline__ uint32_t atom_and_rel(uint32_t* p, uint32_t v) {
  uint32_t r;
  asm volatile("atom.release.gpu.global.and.b32 %0, [%1], %2;" : "=r"(r) : "l"(p), "r"(v) : "memory");
  return r;
}
__device__ __forceinline__ uint32_t atom_or_rel(uint32_t* p, uint32_t v) {
  uint32_t r;
  asm volatile("atom.release.gpu.global.or.b32 %0, [%1], %2;" : "=r"(r) : "l"(p), "r"(v) : "memory");
  return r;
}
__device__ __forceinline__ uint32_t atom_cas(uint32_t* p, uint32_t cmp, uint32_t val) {
  uint32_t r;
  asm volatile("atom.acq_rel.gpu.global.cas.b32 %0, [%1], %2, %3;"
               : "=r"(r) : "l"(p), "r"(cmp), "r"(val) : "memory");
  return r;
}
// Relaxed, fence-free variants for the cache-hit fast path. On sm_100a an
// acquire load/atomic compiles to LDG.STRONG + CCTL.IVALL (invalidates the
// whole L1 of the SM) and a release to MEMBAR.ALL.GPU; the fast path instead
// orders by address dependency and does all metadata accesses at L2.
__device__ __forceinline__ uint32_t atom_add_rlx(uint32_t* p, uint32_t v) {
  uint32_t r;
  asm volatile("atom.relaxed.gpu.global.add.u32 %0, [%1], %2;" : "=r"(r) : "l"(p), "r"(v) : "memory");
  return r;
}
__device__ __forceinline__ void red_add_rlx(uint32_t* p, uint32_t v) {
  asm volatile("red.relaxed.gpu.global.add.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ void red_add64(unsigned long long* p, unsigned long long v) {
  asm volatile("red.relaxed.gpu.global.add.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ unsigned long long atom_add64(unsigned long long* p, unsigned long long v) {
  unsigned long long r;
  asm volatile("atom.relaxed.gpu.global.add.u64 %0, [%1], %2;" : "=l"(r) : "l"(p), "l"(v) : "memory");
  return r;
}
// 64-bit frame-state / tree-slot atomics (generation << 32 | low word)
__device__ __forceinline__ uint64_t a64_add_rlx(uint64_t* p, uint64_t v) {
  uint64_t r;
  asm volatile("atom.relaxed.gpu.global.add.u64 %0, [%1], %2;" : "=l"(r) : "l"(p), "l"(v) : "memory");
  return r;
}
__device__ __forceinline__ uint64_t a64_add_acq(uint64_t* p, uint64_t v) {
  uint64_t r;
  asm volatile("atom.acquire.gpu.global.add.u64 %0, [%1], %2;" : "=l"(r) : "l"(p), "l"(v) : "memory");
  return r;
}
__device__ __forceinline__ uint64_t a64_add_rel(uint64_t* p, uint64_t v) {
  uint64_t r;
  asm volatile("atom.release.gpu.global.add.u64 %0, [%1], %2;" : "=l"(r) : "l"(p), "l"(v) : "memory");
  return r;
}
__device__ __forceinline__ void r64_add_rlx(uint64_t* p, uint64_t v) {
  asm volatile("red.relaxed.gpu.global.add.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ uint64_t a64_and_rel(uint64_t* p, uint64_t v) {
  uint64_t r;
  asm volatile("atom.release.gpu.global.and.b64 %0, [%1], %2;" : "=l"(r) : "l"(p), "l"(v) : "memory");
  return r;
}
__device__ __forceinline__ uint64_t a64_or_rel(uint64_t* p, uint64_t v) {
  uint64_t r;
  asm volatile("atom.release.gpu.global.or.b64 %0, [%1], %2;" : "=l"(r) : "l"(p), "l"(v) : "memory");
  return r;
}
__device__ __forceinline__ uint64_t a64_cas(uint64_t* p, uint64_t cmp, uint64_t val) {
  uint64_t r;
  asm volatile("atom.acq_rel.gpu.global.cas.b64 %0, [%1], %2, %3;"
               : "=l"(r) : "l"(p), "l"(cmp), "l"(val) : "memory");
  return r;
}
// System-scope variants for another GPU's cache (peer fill): the peer's frame
// state words are updated by that GPU's threads; NVLink atomics resolve at
// the owner's L2, and acquire/release must cover both GPUs (.sys).
__device__ __forceinline__ uint64_t ld_rlx_sys64(const uint64_t* p) {
  uint64_t v;
  asm volatile("ld.relaxed.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ uint32_t ld_rlx_sys(const uint32_t* p) {
  uint32_t v;
  asm volatile("ld.relaxed.sys.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ uint64_t a64_add_sys(uint64_t* p, uint64_t v) {
  uint64_t r;
  asm volatile("atom.relaxed.sys.global.add.u64 %0, [%1], %2;" : "=l"(r) : "l"(p), "l"(v) : "memory");
  return r;
}
__device__ __forceinline__ void fence_sys() { asm volatile("fence.acq_rel.sys;" ::: "memory"); }
constexpr uint64_t kRefDec = ~0ull;  // ref - 1 (never borrows: the ref being dropped is >= 1)
__device__ __forceinline__ uint64_t fl64(uint32_t flags) { return ~(uint64_t)flags; }  // and-mask clearing flags
// Leaf slot value for frame f of generation gen.
__device__ __forceinline__ uint64_t slot_val(uint32_t f, uint32_t gen) { return ((uint64_t)gen << 32) | (f + 1u); }
// Bit 31 of a leaf slot's low word: the slot was installed and no lookup has yet
// seen its frame's fill complete. Installs write slot_val_fill(); the first
// lookup that validates the frame (same generation, no FILLING) clears it.
// A slot without the bit therefore names an incarnation whose bytes were
// complete before the slot was read (FILLING is set once per generation, at
// install, and cleared once): gread's one-page fast path may start its copy
// from such a frame before its reference is confirmed (the reference then
// decides whether the copy is kept, gread_t).
constexpr uint32_t kSlotFill = 0x80000000u;
__device__ __forceinline__ uint64_t slot_val_fill(uint32_t f, uint32_t gen) { return slot_val(f, gen) | kSlotFill; }
__device__ __forceinline__ uint32_t slot_frame(uint64_t s) { return ((uint32_t)s & ~kSlotFill) - 1u; }
// Claim frame f for exclusive use (EVICTING) if its low word is exactly `low`
// (0: unreferenced, no flags). Keeps the generation.
__device__ __forceinline__ bool claim_frame(uint64_t* st, uint32_t low) {
  const uint64_t v = ld_rlx64(st);
  if ((uint32_t)v != low) return false;
  return a64_cas(st, v, (v & 0xFFFFFFFF00000000ull) | GFS_ST_EVICTING) == v;
}

__device__ __forceinline__ void backoff(uint32_t& ns) {
  __nanosleep(ns);
  ns = ns < 4096 ? ns * 2 : 4096;
}

__device__ __forceinline__ void ctr(const gfs_ctx* c, int i, unsigned long long v = 1) {
#ifndef GFS_NO_COUNTERS  // (diagnostic builds only: measures what the statistics cost)
  red_add64(&c->ctr[(size_t)i * GFS_CTR_SHARDS + (smid() & (GFS_CTR_SHARDS - 1))], v);
#endif
}

__device__ __forceinline__ uint32_t stamp_now() { return (uint32_t)(now_ns() >> 10); }

__device__ __forceinline__ bool timed_out(const gfs_ctx* c, uint64_t t0) {
  return c->timeout_ns && now_ns() - t0 > c->timeout_ns;
}

// ------------------------------------------------------------------ thread ids
__device__ __forceinline__ int block_tid() {
  return threadIdx.x + blockDim.x * (threadIdx.y + blockDim.y * threadIdx.z);
}
__device__ __forceinline__ int block_nthr() { return blockDim.x * blockDim.y * blockDim.z; }
__device__ __forceinline__ uint64_t grid_id() {
  uint64_t g;
  asm volatile("mov.u64 %0, %%gridid;" : "=l"(g));
  return g;
}
__device__ __forceinline__ uint32_t block_linear() {
  return blockIdx.x + gridDim.x * (blockIdx.y + gridDim.y * blockIdx.z);
}

// ------------------------------------------------------------------ scratch
struct FileSnap {
  uint32_t fdx, uid, root, height, hfid, oflags;
  uint64_t size;
};

struct Scratch {
  int64_t ret;
  int64_t aux;
  void* ptr;
  FileSnap fs;
  // Snapshot of the fd this block opened last: valid while the block holds it
  // open (an open file cannot be re-incarnated). Shared memory is not cleared
  // between launches or blocks, so the key includes %gridid and the block id.
  FileSnap cached;
  uint64_t cached_grid;
  uint32_t cached_blk;
  int32_t cached_fd;
  // Leaf-node ids of the cached file's radix tree, direct-mapped by page >> 8:
  // interior nodes never change while the file is open, so a block that holds
  // it skips the upper levels of the walk (one dependent L2 load fewer).
  // Entries are ((page >> 8) + 1) << 32 | node, one 64-bit store each.
  uint64_t leaf[kLeafCache];
  uint32_t lc_ok;  // this call's snapshot is the cached one (leaf cache usable)
  // mbarrier for TMA bulk copies into shared memory (same validity key)
  uint64_t mbar;
  uint64_t mbar_grid;
  uint32_t mbar_blk;
  uint32_t mbar_phase;
  uint32_t quick;  // this gread's one-page TMA copy was issued by lane 0 before the barrier
  int32_t frame[GFS_MAX_BATCH];   // >= 0 held frame; kBusy / -errno otherwise
  int32_t stage[GFS_MAX_BATCH];   // staging slot to pull from (>= 0), or -1
  uint32_t fill[GFS_MAX_BATCH];   // 1: this block installed the frame and must fill it
  uint32_t nbytes[GFS_MAX_BATCH]; // valid bytes of a filled page
  uint32_t lo[GFS_MAX_BATCH], hi[GFS_MAX_BATCH];
  int32_t err;
  uint32_t busy;
  // read-ahead (NEXT-2), valid for ra_grid / ra_blk: the block's last gread
  // (fd, end), the highest page fetched ahead, and the fills it posted that
  // nobody has completed yet (frame, f_pf value), reaped at gclose
  uint64_t ra_grid;
  uint32_t ra_blk;
  int32_t ra_fd;
  uint64_t ra_next;
  uint64_t ra_hi;
  uint32_t ra_n;
  uint32_t ra_f[16];
  uint64_t ra_v[16];
  // next-call hint (gread_hint): a page of the block's next gread, looked up
  // whose leaf slot was read while this call's copy was in flight (no
  // reference is taken); valid for hint_grid / hint_blk while hint_ok
  uint64_t hint_grid;
  uint32_t hint_blk;
  int32_t hint_fd;
  uint32_t hint_ok;
  uint64_t hint_page;
  uint64_t hint_sv;
};
constexpr uint32_t kRA = 16;  // read-ahead fills a block tracks

__device__ __forceinline__ Scratch& scratch() {
  __shared__ Scratch s;
  return s;
}

// Call groups. The paper's design point is a warp-level API; its
// prototype calls per threadblock. Both share one implementation,
// parameterised by the group: who takes part, how it synchronises, and where
// its scratch lives. key() identifies the group within a launch (scratch is
// shared memory, never cleared, so cached state is keyed by grid and group).
struct BlockGroup {
  static constexpr bool kBlock = true;
  static __device__ __forceinline__ int tid() { return block_tid(); }
  static __device__ __forceinline__ int nthr() { return block_nthr(); }
  static __device__ __forceinline__ void sync() { __syncthreads(); }
  static __device__ __forceinline__ Scratch& sc() { return scratch(); }
  static __device__ __forceinline__ uint32_t key() { return block_linear(); }
};

#ifndef GFS_WARP_API_MAX_WARPS
#define GFS_WARP_API_MAX_WARPS 8  // warp-API blocks have at most 8 warps (scratch: 8 x ~1.2 KiB)
#endif
__device__ __forceinline__ Scratch& warp_scratch(int w) {
  __shared__ Scratch s[GFS_WARP_API_MAX_WARPS];
  return s[w];
}
struct WarpGroup {  // every lane of the calling warp takes part (full warps only)
  static constexpr bool kBlock = false;
  static __device__ __forceinline__ int tid() { return block_tid() & 31; }
  static __device__ __forceinline__ int nthr() { return 32; }
  static __device__ __forceinline__ void sync() { __syncwarp(); }
  static __device__ __forceinline__ Scratch& sc() { return warp_scratch(block_tid() >> 5); }
  static __device__ __forceinline__ uint32_t key() { return (block_linear() << 3) | (uint32_t)(block_tid() >> 5); }
};

// ------------------------------------------------------------------ staging slots
// Pinned host memory, page_size bytes per slot, device-mapped; a bitmap in HBM
// hands slots out. A slot is held only across one RPC and the copy around it,
// never while waiting on another block, so allocation always makes progress.
// wait = false: one pass over the bitmap, -EAGAIN when every slot is taken.
__device__ int stage_alloc(const gfs_ctx* c, bool wait = true) {
  const uint32_t W = c->staging_words;
  uint32_t w = (smid() * 7u + (uint32_t)(now_ns() >> 6)) % W;
  const uint64_t t0 = now_ns();
  uint32_t ns = 64;
  bool waited = false;
  for (uint32_t pass = 0;; ++pass) {
    for (uint32_t k = 0; k < W; ++k, w = (w + 1 == W ? 0 : w + 1)) {
      uint32_t cur = ld_rlx(c->staging_bits + w);
      while (cur != 0xFFFFFFFFu) {
        const uint32_t bit = __ffs(~cur) - 1;
        const uint32_t idx = w * 32 + bit;
        if (idx >= c->staging_slots) break;
        const uint32_t prev = atomicOr(c->staging_bits + w, 1u << bit);
        if (!(prev & (1u << bit))) {
          if (waited) ctr(c, GFS_C_STAGE_WAIT);
          return (int)idx;
        }
        cur = prev | (1u << bit);
      }
    }
    if (!wait) return -EAGAIN;
    waited = true;
    backoff(ns);
    if (timed_out(c, t0)) return -ETIMEDOUT;
  }
}
__device__ __forceinline__ void stage_free(const gfs_ctx* c, int idx) {
  atomicAnd(c->staging_bits + (idx >> 5), ~(1u << (idx & 31)));
}
__device__ __forceinline__ uint8_t* stage_ptr(const gfs_ctx* c, int idx) {
  return c->staging + ((size_t)idx << c->page_shift);
}

// ------------------------------------------------------------------ RPC client
// One request on the per-GPU queue: take a ticket, fill the 64-byte
// slot in pinned host memory, publish seq with st.release.sys (the GPU->CPU
// fence), then poll the completion word the host stores in pinned
// memory (ld.acquire.sys: P:L693-696's cache bypass). Any thread may call.
// rpc_post + rpc_complete are the two halves (read-ahead posts and lets any
// thread complete later); rpc_call is both. Returns the ticket, or -ETIMEDOUT.
__device__ int64_t rpc_post(const gfs_ctx* c, uint32_t op, uint32_t hfid, uint64_t file_off, int stage, uint32_t len,
                            uint32_t flags, uint64_t arg, const char* path, uint32_t path_len) {
  const unsigned long long t = atom_add64(c->ring_tail, 1ull);
  const uint32_t R = c->ring_slots;
  const uint32_t slot = (uint32_t)(t % R);
  const uint64_t t0 = now_ns();
  uint32_t ns = 32;
  if (t >= R) {  // slot reuse: its previous client must have released it
    const uint64_t need = (uint64_t)(t - R + 1);
    bool waited = false;
    while (ld_acq64(&c->ack[slot]) != need) {
      waited = true;
      backoff(ns);
      if (timed_out(c, t0)) {
        ctr(c, GFS_C_TIMEOUT);
        return -ETIMEDOUT;
      }
    }
    if (waited) ctr(c, GFS_C_RING_WAIT);
  }
  volatile gfs_rpc_req* q = c->ring + slot;
  q->op = op;
  q->hfid = hfid;
  q->file_off = file_off;
  q->dev_ptr = 0;
  q->len = len;
  q->flags = flags;
  q->arg = arg;
  q->path_len = path_len;
  q->stage = (uint32_t)stage;
  if (path) {  // 8-byte stores where aligned: each store is one PCIe write
    volatile char* dp = c->ring_paths + (size_t)slot * GFS_MAX_PATH;
    uint32_t i = 0;
    if (((uintptr_t)path & 7) == 0) {
      volatile uint64_t* d8 = (volatile uint64_t*)dp;
      const uint64_t* s8 = (const uint64_t*)path;
      for (; i + 8 <= path_len; i += 8) d8[i >> 3] = s8[i >> 3];
    }
    for (; i < path_len; ++i) dp[i] = path[i];
  }
  st_rel_sys64((uint64_t*)&q->seq, (uint64_t)(t + 1));
  ctr(c, GFS_C_RPC);
  return (int64_t)t;
}

// Wait for ticket t's completion, read its result (and the reply record), and
// release the ring slot to the ticket's successor.
__device__ int32_t rpc_complete(const gfs_ctx* c, uint64_t t, gfs_rpc_resp* resp_out) {
  const uint32_t slot = (uint32_t)(t % c->ring_slots);
  const uint32_t want = (uint32_t)(t + 1);
  const uint64_t t0 = now_ns();
  uint64_t v;
  uint32_t ns = 256;
  while (((v = ld_acq_sys64(&c->cpl[slot])) >> 32) != want) {
    backoff(ns);
    if (timed_out(c, t0)) {
      ctr(c, GFS_C_TIMEOUT);
      // release the slot anyway: the ticket's successor waits for this ack, and
      // a late completion of this ticket carries its own sequence number (the
      // successor waits for t + R + 1), so it cannot be taken for the next one
      st_rel64(&c->ack[slot], (uint64_t)(t + 1));
      return -ETIMEDOUT;
    }
  }
  const int32_t res = (int32_t)(uint32_t)(v & 0xFFFFFFFFull);
  if (resp_out) {
    volatile gfs_rpc_resp* r = c->resp + slot;
    resp_out->size = r->size;
    resp_out->version = r->version;
    resp_out->ino = r->ino;
    resp_out->dev = r->dev;
    resp_out->mtime_ns = r->mtime_ns;
    resp_out->hfid = r->hfid;
    resp_out->status = r->status;
    resp_out->pad[0] = r->pad[0];  // OPEN: bytes of page 0 prefetched into the staging slot
    resp_out->pad[1] = r->pad[1];  // OPEN: device address of the registered file mapping (0: none)
  }
  st_rel64(&c->ack[slot], (uint64_t)(t + 1));
  return res;
}

__device__ int32_t rpc_call(const gfs_ctx* c, uint32_t op, uint32_t hfid, uint64_t file_off, int stage,
                            uint32_t len, uint32_t flags, uint64_t arg, const char* path, uint32_t path_len,
                            gfs_rpc_resp* resp_out) {
  const int64_t t = rpc_post(c, op, hfid, file_off, stage, len, flags, arg, path, path_len);
  if (t < 0) return (int32_t)t;
  return rpc_complete(c, (uint64_t)t, resp_out);
}

// ------------------------------------------------------------------ radix nodes
__device__ __forceinline__ void spin_lock(uint32_t* l) {
  uint32_t ns = 32;
  while (atom_cas(l, 0u, 1u) != 0u) backoff(ns);
}
__device__ __forceinline__ void spin_unlock(uint32_t* l) { st_rel(l, 0u); }

// Returns a zeroed node index (>= 1; node 0 is reserved as "null"), or 0.
// Never-used nodes come from a lock-free bump counter (every first gopen
// needs a root: a source tree opens tens of thousands of files at once);
// recycled nodes from a locked stack.
__device__ uint32_t node_alloc(const gfs_ctx* c) {
  if (ld_rlx(c->node_next) < c->max_nodes) {
    const uint32_t n = atomicAdd(c->node_next, 1u);
    if (n < c->max_nodes) {
      ctr(c, GFS_C_NODES);
      return n;
    }
  }
  uint32_t n = 0;
  spin_lock(c->node_lock);
  uint32_t top = *(volatile uint32_t*)c->node_free_top;
  if (top > 0) {
    n = c->node_free[top - 1];
    *(volatile uint32_t*)c->node_free_top = top - 1;
  }
  spin_unlock(c->node_lock);
  if (n) ctr(c, GFS_C_NODES);
  return n;
}

__device__ void node_free_one(const gfs_ctx* c, uint32_t n) {
  uint4* p = (uint4*)(c->nodes + (size_t)n * GFS_FANOUT);
  for (int i = 0; i < (int)(GFS_FANOUT / 2); ++i) p[i] = make_uint4(0, 0, 0, 0);
  __threadfence();
  spin_lock(c->node_lock);
  uint32_t top = *(volatile uint32_t*)c->node_free_top;
  c->node_free[top] = n;
  *(volatile uint32_t*)c->node_free_top = top + 1;
  spin_unlock(c->node_lock);
}

// Free every node of a tree (caller guarantees no walker: the file is not open).
__device__ void tree_free(const gfs_ctx* c, uint32_t root, uint32_t height) {
  if (!root) return;
  uint32_t stk_node[GFS_MAX_HEIGHT];
  uint32_t stk_idx[GFS_MAX_HEIGHT];
  int sp = 0;
  stk_node[0] = root;
  stk_idx[0] = 0;
  while (sp >= 0) {  // stack depth d holds a node of height (height - d)
    const uint32_t node = stk_node[sp];
    const uint32_t h = height - (uint32_t)sp;
    if (h > 1 && stk_idx[sp] < GFS_FANOUT) {
      const uint32_t i = stk_idx[sp]++;
      const uint32_t ch = (uint32_t)c->nodes[(size_t)node * GFS_FANOUT + i];
      if (ch) {
        ++sp;
        stk_node[sp] = ch;
        stk_idx[sp] = 0;
      }
      continue;
    }
    node_free_one(c, node);
    --sp;
  }
}

// Walk (creating interior nodes if `create`) to the leaf slot of `page`.
// Interior entries hold child node ids; leaf entries hold slot_val(frame, gen).
// New nodes are zeroed before the publishing CAS.
__device__ uint64_t* walk(const gfs_ctx* c, uint32_t root, uint32_t height, uint64_t page, bool create,
                          int* err) {
  uint32_t node = root;
  for (int lvl = (int)height - 1; lvl >= 1; --lvl) {
    const uint32_t idx = (uint32_t)(page >> (GFS_FANOUT_SHIFT * lvl)) & (GFS_FANOUT - 1);
    uint64_t* sp = c->nodes + (size_t)node * GFS_FANOUT + idx;
    uint32_t ch = (uint32_t)ld_acq64(sp);
    if (!ch) {
      if (!create) return nullptr;
      const uint32_t n = node_alloc(c);
      if (!n) {
        if (err) *err = -ENOMEM;
        return nullptr;
      }
      __threadfence();
      const uint32_t prev = (uint32_t)a64_cas(sp, 0ull, n);
      if (prev) {
        node_free_one(c, n);
        ch = prev;
      } else {
        ch = n;
      }
    }
    node = ch;
  }
  return c->nodes + (size_t)node * GFS_FANOUT + (uint32_t)(page & (GFS_FANOUT - 1));
}

__device__ __forceinline__ uint32_t height_for(uint64_t npages) {
  if (npages <= (1ull << 8)) return 1;
  if (npages <= (1ull << 16)) return 2;
  if (npages <= (1ull << 24)) return 3;
  return 4;
}

// ------------------------------------------------------------------ copies
// Block-cooperative copy of n bytes. Frame reads bypass L1 (ld.global.cg):
// a frame may have been refilled since this SM last cached it.
// 16-byte vectors with 4 loads in flight per thread when src/dst are
// co-aligned; 4-byte or byte fallback otherwise.
template <bool kHostSrc>
__device__ __forceinline__ uint8_t ld_b(const uint8_t* p) {
  return kHostSrc ? __ldcv(p) : __ldcg(p);
}
template <bool kHostSrc>
__device__ __forceinline__ int4 ld_v(const int4* p) {
  return kHostSrc ? __ldcv(p) : __ldcg(p);
}
template <bool kHostSrc>
__device__ __forceinline__ uint32_t ld_w(const uint32_t* p) {
  return kHostSrc ? __ldcv(p) : __ldcg(p);
}

template <bool kHostSrc = false>
__device__ __forceinline__ void block_copy_from_frame(uint8_t* dst, const uint8_t* src, uint64_t n, int tid,
                                                      int nthr) {
  if (n == 0) return;
  if ((((uintptr_t)src ^ (uintptr_t)dst) & 15) == 0) {
    const uint64_t h0 = (16 - ((uintptr_t)src & 15)) & 15;
    const uint64_t head = h0 < n ? h0 : n;
    for (uint64_t i = tid; i < head; i += nthr) dst[i] = ld_b<kHostSrc>(src + i);
    const uint64_t nv = (n - head) >> 4;
    const int4* s4 = (const int4*)(src + head);
    int4* d4 = (int4*)(dst + head);
    uint64_t i = tid;
    const uint64_t stride = (uint64_t)nthr;
    for (; i + 3 * stride < nv; i += 4 * stride) {
      int4 a = ld_v<kHostSrc>(s4 + i), b = ld_v<kHostSrc>(s4 + i + stride),
           cc = ld_v<kHostSrc>(s4 + i + 2 * stride), d = ld_v<kHostSrc>(s4 + i + 3 * stride);
      d4[i] = a;
      d4[i + stride] = b;
      d4[i + 2 * stride] = cc;
      d4[i + 3 * stride] = d;
    }
    for (; i < nv; i += stride) d4[i] = ld_v<kHostSrc>(s4 + i);
    const uint64_t done = head + (nv << 4);
    for (uint64_t k = done + tid; k < n; k += nthr) dst[k] = ld_b<kHostSrc>(src + k);
  } else if ((((uintptr_t)src ^ (uintptr_t)dst) & 3) == 0) {
    const uint64_t h0 = (4 - ((uintptr_t)src & 3)) & 3;
    const uint64_t head = h0 < n ? h0 : n;
    for (uint64_t i = tid; i < head; i += nthr) dst[i] = ld_b<kHostSrc>(src + i);
    const uint64_t nw = (n - head) >> 2;
    const uint32_t* s4 = (const uint32_t*)(src + head);
    uint32_t* d4 = (uint32_t*)(dst + head);
    for (uint64_t i = tid; i < nw; i += nthr) d4[i] = ld_w<kHostSrc>(s4 + i);
    for (uint64_t k = head + (nw << 2) + tid; k < n; k += nthr) dst[k] = ld_b<kHostSrc>(src + k);
  } else {
    for (uint64_t i = tid; i < n; i += nthr) dst[i] = ld_b<kHostSrc>(src + i);
  }
}

// Copy into a frame or staging slot from user data / a frame (plain loads).
__device__ __forceinline__ void block_copy_plain(uint8_t* dst, const uint8_t* src, uint64_t n, int tid, int nthr) {
  if (n == 0) return;
  if ((((uintptr_t)src ^ (uintptr_t)dst) & 15) == 0) {
    const uint64_t h0 = (16 - ((uintptr_t)src & 15)) & 15;
    const uint64_t head = h0 < n ? h0 : n;
    for (uint64_t i = tid; i < head; i += nthr) dst[i] = src[i];
    const uint64_t nv = (n - head) >> 4;
    const int4* s4 = (const int4*)(src + head);
    int4* d4 = (int4*)(dst + head);
    for (uint64_t i = tid; i < nv; i += nthr) d4[i] = s4[i];
    for (uint64_t k = head + (nv << 4) + tid; k < n; k += nthr) dst[k] = src[k];
  } else {
    for (uint64_t i = tid; i < n; i += nthr) dst[i] = src[i];
  }
}

__device__ __forceinline__ void block_zero(uint8_t* dst, uint64_t n, int tid, int nthr) {
  const uint64_t h0 = (16 - ((uintptr_t)dst & 15)) & 15;
  const uint64_t head = h0 < n ? h0 : n;
  for (uint64_t i = tid; i < head; i += nthr) dst[i] = 0;
  const uint64_t nv = (n - head) >> 4;
  int4* d4 = (int4*)(dst + head);
  for (uint64_t k = tid; k < nv; k += nthr) d4[k] = make_int4(0, 0, 0, 0);
  for (uint64_t k = head + (nv << 4) + tid; k < n; k += nthr) dst[k] = 0;
}

// ------------------------------------------------------------------ TMA bulk copy
// cp.async.bulk global -> shared, completion counted in bytes on an mbarrier
// (SASS UBLKCP). Used by gread when the destination is shared memory: one
// thread moves the whole span, the data never passes through registers.
__device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ void mbar_init(uint64_t* m) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(smem_u32(m)) : "memory");
  asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
}
__device__ __forceinline__ void mbar_expect_tx(uint64_t* m, uint32_t bytes) {
  asm volatile("{ .reg .b64 st; mbarrier.arrive.expect_tx.shared::cta.b64 st, [%0], %1; }" ::"r"(smem_u32(m)),
               "r"(bytes) : "memory");
}
__device__ __forceinline__ void tma_load(void* dst_smem, const void* src, uint32_t bytes, uint64_t* m) {
  asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                   smem_u32(dst_smem)),
               "l"(src), "r"(bytes), "r"(smem_u32(m))
               : "memory");
}
__device__ __forceinline__ void mbar_wait(uint64_t* m, uint32_t phase) {
  asm volatile(
      "{ .reg .pred P1;\n"
      "WAIT_%=: mbarrier.try_wait.parity.shared::cta.b64 P1, [%0], %1;\n"
      "@!P1 bra WAIT_%=;\n}" ::"r"(smem_u32(m)),
      "r"(phase)
      : "memory");
}

// The block's mbarrier lives in `Scratch` (static shared memory, not cleared
// between launches): (re)initialise it the first time this block of this launch
// needs it. Called by thread 0 only, before the barrier that publishes it.
template <class G = BlockGroup>
__device__ __forceinline__ void ensure_mbar(Scratch& sc) {
  if (sc.mbar_grid != grid_id() || sc.mbar_blk != G::key()) {
    mbar_init(&sc.mbar);
    sc.mbar_phase = 0;
    sc.mbar_grid = grid_id();
    sc.mbar_blk = G::key();
  }
}

// TMA bulk copy of one co-aligned span ((dst - src) % 16 == 0): the 16-byte
// aligned middle goes through cp.async.bulk, the <16-byte head and tail are
// left to copy_edges(). Returns the bytes the mbarrier must expect.
__device__ __forceinline__ uint32_t span_mid(const uint8_t* src, uint32_t n) {
  const uint32_t h0 = (16u - ((uint32_t)(uintptr_t)src & 15u)) & 15u;
  return (n - (h0 < n ? h0 : n)) & ~15u;
}
__device__ __forceinline__ uint32_t tma_span(uint8_t* dst, const uint8_t* src, uint32_t n, uint64_t* m) {
  const uint32_t h0 = (16u - ((uint32_t)(uintptr_t)src & 15u)) & 15u;
  const uint32_t head = h0 < n ? h0 : n;
  const uint32_t mid = (n - head) & ~15u;
  if (mid) tma_load(dst + head, src + head, mid, m);
  return mid;
}

// The head and tail bytes tma_span() leaves out, copied by threads tid < 32.
__device__ __forceinline__ void copy_edges(uint8_t* dst, const uint8_t* src, uint32_t n, int tid) {
  const uint32_t h0 = (16u - ((uint32_t)(uintptr_t)src & 15u)) & 15u;
  const uint32_t head = h0 < n ? h0 : n;
  const uint32_t mid = (n - head) & ~15u;
  const uint32_t tail = n - head - mid;
  if (tid < (int)head) dst[tid] = __ldcg(src + tid);
  else if (tid < (int)(head + tail)) {
    const uint32_t k = head + mid + (uint32_t)tid - head;
    dst[k] = __ldcg(src + k);
  }
}

// ------------------------------------------------------------------ frames
__device__ __forceinline__ uint8_t* frame_ptr(const gfs_ctx* c, uint32_t f) {
  return c->pool + ((size_t)f << c->page_shift);
}

// Returns the frame's new generation (the value its tree slot must carry).
__device__ __forceinline__ uint32_t frame_init(const gfs_ctx* c, uint32_t f, uint64_t tag, uint32_t fdx) {
  st_rlx64(&c->f_tag[f], tag);
  st_rlx(&c->f_file[f], fdx);
  st_rlx(&c->f_valid[f], 0);
  st_rlx(&c->f_lo[f], GFS_DIRTY_NONE);
  st_rlx(&c->f_hi[f], 0);
  st_rlx(&c->f_written[f], 0);
  st_rlx(&c->f_hv[f], 0);
  st_rlx(&c->f_pristine[f], 0);
  st_rlx(&c->f_stamp[f], stamp_now());
  // EVICTING -> FILLING|1 and generation + 1 as one atomic delta: readers that
  // found the frame through a stale slot may hold transient +1s they are about
  // to undo, so the state word is never overwritten with a plain store.
  const uint64_t delta = (1ull << 32) + (uint64_t)GFS_ST_FILLING + 1ull - (uint64_t)GFS_ST_EVICTING;
  return (uint32_t)((a64_add_rel(&c->f_state[f], delta) + delta) >> 32);
}

// After a successful write-back of [lo, hi) (wr bytes written) that left the
// host file at `version`: a frame written from byte 0 without holes now equals
// the host file on [0, hi) (host-verified prefix, peer fill), and the file's
// synced version advances.
__device__ __forceinline__ void synced(const gfs_ctx* c, uint32_t f, uint32_t lo, uint32_t hi, uint32_t wr,
                                       uint64_t version) {
  st_rlx(&c->f_hv[f], (lo == 0 && wr >= hi) ? hi : 0u);
  const uint32_t fi = ld_rlx(&c->f_file[f]);
  if (fi < c->max_files) atomicMax((unsigned long long*)&c->files[fi].synced_version, (unsigned long long)version);
}

// Drop the page a published frame holds: tag cleared, generation + 1 (every
// tree slot naming the old generation is now stale), `flag` (held by the
// caller) cleared, in one atomic delta.
__device__ __forceinline__ void frame_retire(const gfs_ctx* c, uint32_t f, uint32_t flag) {
  st_rlx64(&c->f_tag[f], GFS_TAG_NONE);
  a64_add_rel(&c->f_state[f], (1ull << 32) - (uint64_t)flag);
}

// O_RDWR: drop frame f's pristine copy (after its diff was
// written back). The pristine frame was held FILLING|1 (never evictable).
__device__ __forceinline__ void pristine_free(const gfs_ctx* c, uint32_t f) {
  const uint32_t pv = ld_rlx(&c->f_pristine[f]);
  if (pv == 0 || pv == GFS_PRISTINE_PENDING) return;
  st_rlx(&c->f_pristine[f], 0);
  const uint32_t pf = pv - 1;
  frame_retire(c, pf, GFS_ST_FILLING);   // generation + 1, tag none
  a64_add_rel(&c->f_state[pf], kRefDec);  // unreferenced: reclaimable (tier 0)
}

// Write back a frame's dirty range from one thread (the caller owns the frame:
// EVICTING, ref 0): copy it into a staging slot over PCIe, then WRITE RPC.
// nowait: if the staging slots it needs are not free right now, return
// -EAGAIN instead of waiting (eviction: the caller may hold a staging slot of
// its own, so waiting here would be hold-and-wait; it picks another victim).
__device__ __noinline__ int32_t frame_writeback_lane(const gfs_ctx* c, uint32_t f, uint32_t hfid,
                                                     bool nowait = false) {
  const uint32_t lo = ld_rlx(&c->f_lo[f]);
  if (lo == GFS_DIRTY_NONE) return 0;
  const uint32_t hi = ld_rlx(&c->f_hi[f]);
  const uint32_t wr = ld_rlx(&c->f_written[f]);
  const uint64_t page = ld_rlx64(&c->f_tag[f]) & 0xFFFFFFFFull;
  const uint32_t pv = ld_rlx(&c->f_pristine[f]);
  const bool diff = pv != 0 && pv != GFS_PRISTINE_PENDING;  // O_RDWR page: diff against its pristine copy
  int st = -1, st2 = -1;
  const uint64_t t0 = now_ns();
  for (uint32_t ns = 64;;) {  // both slots or none: never wait for one while holding the other
    st = stage_alloc(c, false);
    if (st >= 0 && diff) {
      st2 = stage_alloc(c, false);
      if (st2 < 0) {
        stage_free(c, st);
        st = -1;
      }
    }
    if (st >= 0) break;
    if (nowait) return -EAGAIN;
    backoff(ns);
    if (timed_out(c, t0)) return -ETIMEDOUT;
  }
  // frame bytes via L2 (.cg): this SM's L1 may hold lines of a previous tenant
  block_copy_from_frame(stage_ptr(c, st) + lo, frame_ptr(c, f) + lo, hi - lo, 0, 1);
  if (diff) block_copy_from_frame(stage_ptr(c, st2) + lo, frame_ptr(c, pv - 1) + lo, hi - lo, 0, 1);
  __threadfence_system();
  gfs_rpc_resp rs;
  const int32_t r = rpc_call(c, GFS_OP_WRITE, hfid, (page << c->page_shift) + lo, st, hi - lo,
                             diff ? GFS_WF_DIFF : (wr >= hi - lo ? GFS_WF_FULL : 0u), diff ? (uint64_t)st2 : 0,
                             nullptr, 0, &rs);
  stage_free(c, st);
  if (st2 >= 0) stage_free(c, st2);
  if (r < 0) return r;
  synced(c, f, lo, hi, wr, rs.version);
  if (diff) {
    st_rlx(&c->f_hv[f], 0);
    pristine_free(c, f);
  }
  st_rlx(&c->f_lo[f], GFS_DIRTY_NONE);
  st_rlx(&c->f_hi[f], 0);
  st_rlx(&c->f_written[f], 0);
  ctr(c, GFS_C_WRITEBACK);
  ctr(c, GFS_C_RPC_WRITE);
  ctr(c, GFS_C_BYTES_D2H, hi - lo);
  return 0;
}

// Tier of a reclaimable frame: 0 orphan/invalid/error,
// 1 page of a closed file, 2 clean page of an open file, 3 dirty page.
__device__ __forceinline__ uint32_t frame_tier(const gfs_ctx* c, uint32_t f, uint32_t st) {
  const uint64_t tag = ld_rlx64(&c->f_tag[f]);
  if ((st & GFS_ST_ERROR) || tag == GFS_TAG_NONE) return 0;
  const uint32_t fi = ld_rlx(&c->f_file[f]);
  if (fi >= c->max_files) return 0;
  const gfs_file* e = c->files + fi;
  if (ld_rlx(&e->uid) != (uint32_t)(tag >> 32)) return 0;
  if (ld_rlx(&c->f_lo[f]) != GFS_DIRTY_NONE) return 3;
  if ((ld_rlx(&e->sr) >> 24) == GFS_FS_CLOSED) return 1;
  return 2;
}

// Allocate a frame for `tag`: never-used frames first, else evict the oldest
// reclaimable frame of a 32-frame window (sampled LRU, tiered by P:L651-657),
// writing back a dirty victim first. Runs in the calling thread.
// Returns the frame in state FILLING|1 with its tag set (and its new
// generation in *gen), or -ENOMEM.
__device__ __noinline__ int alloc_frame(const gfs_ctx* c, uint64_t tag, uint32_t fdx, uint32_t* gen,
                                        bool nowait = false) {
  const uint32_t N = c->nframes;
  if (ld_rlx(c->fresh_next) < N) {
    const uint32_t f = atomicAdd(c->fresh_next, 1u);
    if (f < N) {
      *gen = frame_init(c, f, tag, fdx);
      return (int)f;
    }
  }
  const uint64_t t0 = now_ns();
  const uint32_t windows = (N + 31) / 32;
  uint32_t ns = 64;
  for (uint32_t round = 0;; ++round) {
    const uint32_t w = atomicAdd(c->hand, 32u);
    int best = -1;
    uint64_t best_key = ~0ull;
    uint64_t best_st = 0, best_pv = 0;
#pragma unroll 4
    for (uint32_t j = 0; j < 32; ++j) {
      const uint32_t f = (uint32_t)(((uint64_t)w + j) % N);
      const uint64_t st = ld_rlx64(&c->f_state[f]);
      uint64_t pv = 0;
      if ((uint32_t)st & ~GFS_ST_ERROR) {  // referenced, filling or being evicted ...
        // ... except a read-ahead fill nobody has asked for yet (NEXT-2): the
        // last resort (tier 4), so read-ahead never starves a reader of frames
        if (!c->readahead || (uint32_t)st != GFS_ST_FILLING) continue;
        pv = ld_rlx64(&c->f_pf[f]);
        if (pv == 0 || pv == GFS_PF_POSTING) continue;
      }
      const uint64_t key =
          ((uint64_t)(pv ? 4u : frame_tier(c, f, (uint32_t)st)) << 32) | ld_rlx(&c->f_stamp[f]);
      if (key < best_key) {
        best_key = key;
        best = (int)f;
        best_st = st;
        best_pv = pv;
      }
    }
    if (best >= 0 && best_pv) {  // take the unneeded read-ahead fill over and drop its page
      if (a64_cas(&c->f_pf[best], best_pv, 0) != best_pv) continue;  // someone adopted it meanwhile
      (void)rpc_complete(c, (best_pv >> 32) - 1, nullptr);  // the slot and ring entry are released first
      stage_free(c, (int)(uint32_t)best_pv - 1);
      a64_add_rel(&c->f_state[best], (uint64_t)GFS_ST_EVICTING - (uint64_t)GFS_ST_FILLING);  // keeps transient refs
      ctr(c, GFS_C_EVICT);
      *gen = frame_init(c, (uint32_t)best, tag, fdx);
      return best;
    }
    if (best >= 0 &&
        a64_cas(&c->f_state[best], best_st, (best_st & 0xFFFFFFFF00000000ull) | GFS_ST_EVICTING) == best_st) {
      const uint32_t f = (uint32_t)best;
      if (ld_rlx(&c->f_lo[f]) != GFS_DIRTY_NONE) {
        const uint32_t fi = ld_rlx(&c->f_file[f]);
        const int32_t r = frame_writeback_lane(c, f, ld_rlx(&c->files[fi].hfid), true);
        if (r < 0) {  // keep the dirty page, try another victim (no free staging slot: never wait here)
          a64_and_rel(&c->f_state[f], fl64(GFS_ST_EVICTING));
          continue;
        }
      }
      ctr(c, GFS_C_EVICT);
      *gen = frame_init(c, f, tag, fdx);
      return (int)f;
    }
    if (nowait && round >= 8) return -EAGAIN;  // read-ahead: a few windows, never wait for a victim
    if (round > 0 && round % windows == 0) {
      backoff(ns);
      if (now_ns() - t0 > 2000000000ull) {  // 2 s of full scans: the deadlock guard
        ctr(c, GFS_C_ENOMEM);
        return -ENOMEM;
      }
    }
  }
}

// Release after reading a frame: the block barrier before it guarantees every
// load of the frame has returned (its consumer store could not issue
// otherwise), so a relaxed decrement suffices.
__device__ __forceinline__ void frame_release(const gfs_ctx* c, uint32_t f) {
  st_rlx(&c->f_stamp[f], stamp_now());
  r64_add_rlx(&c->f_state[f], kRefDec);  // ref - 1
}
// Release after writing a frame (gwrite): the dirty-range updates must be
// visible before the reference drops (gfsync only syncs unreferenced frames).
__device__ __forceinline__ void frame_release_rel(const gfs_ctx* c, uint32_t f) {
  st_rlx(&c->f_stamp[f], stamp_now());
  a64_add_rel(&c->f_state[f], kRefDec);
}


// Give back a frame we installed but could not publish (lost the CAS race).
__device__ __forceinline__ void frame_abandon(const gfs_ctx* c, uint32_t f) {
  st_rel64(&c->f_tag[f], GFS_TAG_NONE);
  a64_and_rel(&c->f_state[f], fl64(GFS_ST_FILLING));
  a64_add_rel(&c->f_state[f], kRefDec);
}

// ------------------------------------------------------------------ page lookup
// Cache-hit fast path (one optimistic attempt): relaxed walk
// without creating nodes, then ONE relaxed atomic increment of the frame's
// state word that both takes the reference and validates the slot: the
// generation it returns must equal the one stored in the slot (the frame was
// not reassigned since it was installed for this page) and no FILLING /
// EVICTING / ERROR flag may be set. This replaces the paper's tag re-check
// by a per-frame generation, so a hit costs two dependent L2
// round trips instead of three. The tree cannot be freed under us: the
// caller's block holds the file open. All accesses are strong gpu-scope
// operations served at L2, so no L1 line can be stale. Returns the frame, or
// -1 to take the full (acquire/release) path.
// The leaf slot of `page` (relaxed walk, leaf cache), or nullptr when an
// interior node is missing.
__device__ __forceinline__ uint64_t* leaf_slot(const gfs_ctx* c, const FileSnap& fs, uint64_t page,
                                               uint64_t* leaf_cache) {
  uint32_t node = fs.root;
  if (fs.height > 1) {
    const uint32_t key = (uint32_t)(page >> GFS_FANOUT_SHIFT);
    const uint64_t ent = leaf_cache ? leaf_cache[key & (kLeafCache - 1)] : 0;
    if (ent >> 32 == (uint64_t)key + 1) {
      node = (uint32_t)ent;
    } else {
      for (int lvl = (int)fs.height - 1; lvl >= 1; --lvl) {
        node = (uint32_t)ld_rlx64(c->nodes + (size_t)node * GFS_FANOUT +
                                  ((uint32_t)(page >> (GFS_FANOUT_SHIFT * lvl)) & 255u));
        if (!node) return nullptr;
      }
      if (leaf_cache) leaf_cache[key & (kLeafCache - 1)] = (((uint64_t)key + 1) << 32) | node;
    }
  }
  return c->nodes + (size_t)node * GFS_FANOUT + ((uint32_t)page & 255u);
}

__device__ __forceinline__ int lookup_fast(const gfs_ctx* c, const FileSnap& fs, uint64_t page,
                                           uint64_t* leaf_cache = nullptr) {
  uint64_t* const sp = leaf_slot(c, fs, page, leaf_cache);
  if (!sp) return -1;
  const uint64_t s = ld_rlx64(sp);
  if (!(uint32_t)s) return -1;
  const uint32_t f = slot_frame(s);
  const uint64_t old = a64_add_rlx(&c->f_state[f], 1ull);
  if ((old >> 32) == (s >> 32) && !((uint32_t)old & (GFS_ST_FILLING | GFS_ST_EVICTING | GFS_ST_ERROR))) {
    if ((uint32_t)s & kSlotFill) a64_cas(sp, s, s & ~(uint64_t)kSlotFill);  // the fill is complete: say so
    ctr(c, GFS_C_HIT);
    ctr(c, GFS_C_LOCKFREE);
    return (int)f;
  }
  r64_add_rlx(&c->f_state[f], kRefDec);
  return -1;
}

// True if page `page` is installed and currently FILLING or EVICTING (no
// reference taken, no lock): a waiter can keep waiting without contending.
__device__ __forceinline__ bool peek_busy(const gfs_ctx* c, const FileSnap& fs, uint64_t page) {
  uint32_t node = fs.root;
  for (int lvl = (int)fs.height - 1; lvl >= 1; --lvl) {
    node = (uint32_t)ld_rlx64(c->nodes + (size_t)node * GFS_FANOUT +
                              ((uint32_t)(page >> (GFS_FANOUT_SHIFT * lvl)) & 255u));
    if (!node) return false;
  }
  const uint64_t s = ld_rlx64(c->nodes + (size_t)node * GFS_FANOUT + ((uint32_t)page & 255u));
  if (!(uint32_t)s) return false;
  const uint64_t st = ld_rlx64(&c->f_state[slot_frame(s)]);
  return (st >> 32) == (s >> 32) && ((uint32_t)st & (GFS_ST_FILLING | GFS_ST_EVICTING));
}

// ------------------------------------------------------------------ peer fill
// NEXT-1 (the buffer cache spans GPUs). On a miss of
// an O_RDONLY file, before asking the host, look the page up in the peer
// caches (gfs_peer views of other GPUs' caches, mapped over NVLink). A peer
// frame is usable iff it holds the same host file (st_ino, st_dev) at the
// same close-to-open version as this cache's entry, is clean, and its first
// nb bytes are host-verified (f_hv: filled from the host, or written from
// byte 0 without holes and then written back). For a peer's O_GWRONCE entry
// the version is the one its last write-back left (synced_version). Taking
// the peer frame is the hit protocol of lookup_fast run at system scope: one
// atomic increment takes the reference and validates the slot's generation;
// the peer's eviction skips referenced frames. Result code (k << 27) | f, or
// -1 when no peer has a usable copy.
constexpr uint32_t kPeerFrameBits = 27;
__device__ __noinline__ int peer_take(const gfs_ctx* c, const FileSnap& fs, uint64_t page, uint32_t nb) {
  const gfs_file* me = c->files + fs.fdx;
  const uint64_t h = ld_rlx64(&me->path_hash);
  const uint32_t n = ld_rlx(&me->path_len);
  const uint64_t ino = ld_rlx64(&me->ino), dev = ld_rlx64(&me->dev), ver = ld_rlx64(&me->version);
  const int64_t mt = (int64_t)ld_rlx64((const uint64_t*)&me->mtime_ns);
  const uint32_t np = c->npeers;
  for (uint32_t j = 0; j < np; ++j) {
    const uint32_t k = (j + (uint32_t)page) % np;  // spread a sweep's pages over the peers
    const gfs_peer& P = c->peers[k];
    const uint32_t mask = P.max_files - 1u;
    uint32_t i = (uint32_t)h & mask;
    for (uint32_t probe = 0; probe < 64; ++probe, i = (i + 1u) & mask) {
      gfs_file* e = P.files + i;
      const uint32_t st = ld_rlx_sys(&e->sr) >> 24;
      if (st == GFS_FS_FREE) break;
      if (st != GFS_FS_OPEN && st != GFS_FS_CLOSED) continue;
      if (ld_rlx_sys64(&e->path_hash) != h || ld_rlx_sys(&e->path_len) != n) continue;
      if (ld_rlx_sys64(&e->ino) != ino || ld_rlx_sys64(&e->dev) != dev) continue;
      const uint32_t uid = ld_rlx_sys(&e->uid);
      const uint32_t pof = ld_rlx_sys(&e->oflags);
      if (pof & GFS_O_RDWR) break;  // a read-write peer's frames may hold unsynced or diffed bytes
      const bool wonce = (pof & GFS_O_GWRONCE) != 0;
      const uint64_t ev = wonce ? ld_rlx_sys64(&e->synced_version) : ld_rlx_sys64(&e->version);
      if ((wonce && ev == 0) || ev != ver) break;  // the peer's copy is of another version
      if (!wonce && (ld_rlx_sys64(&e->size) != fs.size || (int64_t)ld_rlx_sys64((const uint64_t*)&e->mtime_ns) != mt))
        break;
      const uint32_t height = ld_rlx_sys(&e->height);
      if (height == 0 || height > GFS_MAX_HEIGHT || (height < 4 && (page >> (GFS_FANOUT_SHIFT * height)) != 0)) break;
      uint32_t node = ld_rlx_sys(&e->root);
      for (int lvl = (int)height - 1; lvl >= 1 && node && node < P.max_nodes; --lvl)
        node = (uint32_t)ld_rlx_sys64(P.nodes + (size_t)node * GFS_FANOUT +
                                      ((uint32_t)(page >> (GFS_FANOUT_SHIFT * lvl)) & 255u));
      if (!node || node >= P.max_nodes) break;  // type-stable nodes: a racing free reads as a miss
      const uint64_t sl = ld_rlx_sys64(P.nodes + (size_t)node * GFS_FANOUT + ((uint32_t)page & 255u));
      const uint32_t f = slot_frame(sl);
      if (!(uint32_t)sl || f >= P.nframes) break;
      const uint64_t old = a64_add_sys(&P.f_state[f], 1ull);
      fence_sys();  // the checks and the copy below read after the reference is held
      if ((old >> 32) == (sl >> 32) && !((uint32_t)old & (GFS_ST_FILLING | GFS_ST_EVICTING | GFS_ST_ERROR)) &&
          ld_rlx_sys64(&P.f_tag[f]) == (((uint64_t)uid << 32) | (uint32_t)page) &&
          ld_rlx_sys(&P.f_lo[f]) == GFS_DIRTY_NONE && ld_rlx_sys(&P.f_hv[f]) >= nb)
        return (int)((k << kPeerFrameBits) | f);
      a64_add_sys(&P.f_state[f], kRefDec);
      break;
    }
  }
  ctr(c, GFS_C_PEER_MISS);
  return -1;
}
__device__ __forceinline__ const uint8_t* peer_frame_ptr(const gfs_ctx* c, int code) {
  const gfs_peer& P = c->peers[(uint32_t)code >> kPeerFrameBits];
  return P.pool + ((size_t)((uint32_t)code & ((1u << kPeerFrameBits) - 1u)) << P.page_shift);
}
__device__ __forceinline__ void peer_release(const gfs_ctx* c, int code) {
  const gfs_peer& P = c->peers[(uint32_t)code >> kPeerFrameBits];
  a64_add_sys(&P.f_state[(uint32_t)code & ((1u << kPeerFrameBits) - 1u)], kRefDec);
}
// Lk.stage / Scratch.stage: >= 0 staging slot, -1 nothing to pull, kStageZC
// the file's registered host mapping (zero-copy), other values <= -2 a peer frame
constexpr int kStageZC = -0x7FFFFFFF;
__device__ __forceinline__ int peer_stage(int code) { return -2 - code; }
__device__ __forceinline__ int stage_peer(int stage) { return -2 - stage; }
__device__ __forceinline__ const uint8_t* fill_src(const gfs_ctx* c, int stage, const FileSnap& fs,
                                                   uint64_t page) {
  if (stage == kStageZC) return (const uint8_t*)ld_rlx64(&c->files[fs.fdx].zc) + (page << c->page_shift);
  return stage >= 0 ? stage_ptr(c, stage) : peer_frame_ptr(c, stage_peer(stage));
}
__device__ __forceinline__ void fill_src_free(const gfs_ctx* c, int stage) {
  if (stage == kStageZC) return;
  if (stage >= 0) stage_free(c, stage);
  else peer_release(c, stage_peer(stage));
}

struct Lk {
  int frame;   // >= 0 held (ref taken); kBusy; or -errno
  int stage;   // >= 0: pull nbytes from this staging slot into the frame
  uint32_t fill;
  uint32_t nbytes;
};

// Find page `page` of the snapshot file and take a reference (P:L575-576,
// P:L616-619). Lock-free: read slot, incref, validate tag == (uid,page)
// (P:L669-672). Retries once without locking, then takes the file lock on
// the third attempt. Never waits on another block: a page being
// filled or evicted elsewhere returns kBusy. A miss installs a frame by CAS
// and returns it with fill = 1 and FILLING still set: for O_RDONLY files the
// page has been pread by the host into staging slot `stage` (READ RPC,
// P:L570-576); for O_GWRONCE files nothing is fetched. The
// caller's block fills the frame and clears FILLING.
__device__ __noinline__ Lk lookup_try(const gfs_ctx* c, const FileSnap& fs, uint64_t page) {
  Lk out{kBusy, -1, 0, 0};
  const uint64_t want = ((uint64_t)fs.uid << 32) | (uint32_t)page;
  uint32_t* lockp = &c->files[fs.fdx].lock;
  const bool always_lock = (c->flags & GFS_F_LOCKED_TRAVERSAL) != 0;  // K5 ablation
  bool used_lock = false;
  int attempt = 0;
  uint64_t* slot = nullptr;
  for (;;) {
    // The lock (when taken) covers the traversal only: walk, slot read,
    // reference + validation. Fills and RPCs run unlocked.
    const bool lk = always_lock || attempt >= 2;
    if (lk) {
      spin_lock(lockp);
      used_lock = true;
    }
    if (!slot) {
      int err = 0;
      slot = walk(c, fs.root, fs.height, page, true, &err);
      if (!slot) {
        if (lk) spin_unlock(lockp);
        out.frame = err ? err : -ENOMEM;
        break;
      }
    }
    const uint64_t s = ld_acq64(slot);
    bool done = false;
    if ((uint32_t)s) {
      const uint32_t f = slot_frame(s);
      const uint64_t old = a64_add_acq(&c->f_state[f], 1ull);
      // same generation as the slot <=> the frame still holds this page (the
      // tag check is kept as a belt-and-braces test on the slow path)
      if ((old >> 32) == (s >> 32) && ld_acq64(&c->f_tag[f]) == want) {
        uint64_t pv = 0;
        if (!((uint32_t)old & (GFS_ST_FILLING | GFS_ST_EVICTING | GFS_ST_ERROR))) {
          ctr(c, GFS_C_HIT);
          out.frame = (int)f;
          done = true;
        } else if (!lk && ((uint32_t)old & (GFS_ST_FILLING | GFS_ST_EVICTING)) == GFS_ST_FILLING &&
                   (pv = ld_acq64(&c->f_pf[f])) != 0 && pv != GFS_PF_POSTING && a64_cas(&c->f_pf[f], pv, 0) == pv) {
          // a read-ahead fill nobody waits for yet (NEXT-2): this lane completes
          // it — the host has (or will have) the page in the posted staging
          // slot — and keeps the reference it just took as its own
          const int stg = (int)(uint32_t)pv - 1;
          const int32_t r = rpc_complete(c, (pv >> 32) - 1, nullptr);
          if (r < 0) {  // the fetch failed: the frame becomes stale, retried below like any stale slot
            stage_free(c, stg);
            a64_or_rel(&c->f_state[f], GFS_ST_ERROR);
            a64_and_rel(&c->f_state[f], fl64(GFS_ST_FILLING));
            a64_add_rel(&c->f_state[f], kRefDec);
          } else {
            ctr(c, GFS_C_RA_ADOPTED);
            out.frame = (int)f;
            out.fill = 1;
            out.stage = stg;
            out.nbytes = (uint32_t)r;
            done = true;
          }
        } else if ((uint32_t)old & (GFS_ST_FILLING | GFS_ST_EVICTING)) {  // someone else is on it
          a64_add_rel(&c->f_state[f], kRefDec);
          ctr(c, GFS_C_BUSY);
          out.frame = kBusy;
          done = true;
        } else {
          a64_add_rel(&c->f_state[f], kRefDec);  // ERROR, no fill in flight: stale, install over it
        }
      } else {
        a64_add_rel(&c->f_state[f], kRefDec);  // stale slot: install over it
      }
      if (!done) {
        ++attempt;
        ctr(c, GFS_C_RETRY);
      }
    }
    if (lk) spin_unlock(lockp);
    if (done) break;
    // miss (or stale slot). A fill needs a staging slot: take one BEFORE
    // installing anything, without waiting. If none is free the page is
    // reported busy and retried after this block has pulled (and released)
    // the pages it did install: a lane never waits for a slot while its block
    // holds others (hold-and-wait across blocks deadlocked at small pages).
    const uint64_t base = page << c->page_shift;
    const uint64_t rem = fs.size > base ? fs.size - base : 0;
    const uint32_t nb = (fs.oflags & GFS_O_GWRONCE) ? 0u : (uint32_t)(rem < c->page_size ? rem : c->page_size);
    // A peer GPU's cache may hold the page (NEXT-1): then no staging slot
    // and no RPC; `st` names the peer frame (held) instead.
    // A registered host mapping of the file (gfs_register_file): the block pulls
    // the page straight from the host page cache, no RPC and no staging slot.
    const bool zc = nb && ld_rlx64(&c->files[fs.fdx].zc) != 0;
    const int pc = (nb && !zc && c->npeers) ? peer_take(c, fs, page, nb) : -1;
    int st = -1;
    if (zc) {
      st = kStageZC;
    } else if (pc >= 0) {
      st = peer_stage(pc);
    } else if (nb) {
      st = stage_alloc(c, false);
      if (st < 0) st = -1;  // -EAGAIN: every slot taken
    }
    if (nb && st == -1) {
      ctr(c, GFS_C_STAGE_WAIT);
      out.frame = kBusy;
      break;
    }
    // Install a new frame for `want`. The slot value carries the frame's
    // generation, so the CAS cannot succeed against a value that was replaced
    // and restored in between (no ABA).
    uint32_t gen = 0;
    const int g = alloc_frame(c, want, fs.fdx, &gen);
    if (g < 0) {
      if (st != -1) fill_src_free(c, st);
      out.frame = g;
      break;
    }
    const bool won = a64_cas(slot, s, slot_val_fill((uint32_t)g, gen)) == s;
    if (!won) {
      if (st != -1) fill_src_free(c, st);
      frame_abandon(c, (uint32_t)g);
      ++attempt;
      ctr(c, GFS_C_RETRY);
      continue;
    }
    out.frame = g;
    out.fill = 1;
    if (fs.oflags & GFS_O_GWRONCE) {
      ctr(c, GFS_C_ZERO_FILL);
      break;
    }
    if (zc) {  // the block pulls from the registered mapping over PCIe
      out.stage = st;
      out.nbytes = nb;
      ctr(c, GFS_C_MISS);
      ctr(c, GFS_C_ZC_FILL);
      ctr(c, GFS_C_BYTES_H2D, nb);
      break;
    }
    if (pc >= 0) {  // the block copies the peer frame over NVLink
      out.stage = st;
      out.nbytes = nb;
      ctr(c, GFS_C_PEER_FILL);
      ctr(c, GFS_C_BYTES_PEER, nb);
      break;
    }
    // Fetch min(P, S - pP) bytes: the host preads into the staging slot.
    int32_t r = 0;
    if (nb) r = rpc_call(c, GFS_OP_READ, fs.hfid, base, st, nb, 0, 0, nullptr, 0, nullptr);
    if (r < 0) {
      if (st >= 0) stage_free(c, st);
      a64_or_rel(&c->f_state[g], GFS_ST_ERROR);
      a64_and_rel(&c->f_state[g], fl64(GFS_ST_FILLING));
      a64_add_rel(&c->f_state[g], kRefDec);
      out.frame = r == -ETIMEDOUT ? r : -EIO;
      out.fill = 0;
      break;
    }
    out.stage = st;
    out.nbytes = nb;
    ctr(c, GFS_C_MISS);
    ctr(c, GFS_C_RPC_READ);
    ctr(c, GFS_C_BYTES_H2D, nb);
    break;
  }
  if (used_lock) {
    ctr(c, GFS_C_LOCKED);
  } else if (out.frame >= 0) {
    ctr(c, GFS_C_LOCKFREE);
  }
  return out;
}

// Take references on pages [pb, pb + cnt) (cnt <= 32), all threads calling.
// Lookups run one page per lane of warp 0 (parallel misses = parallel RPCs).
// Pages this block installed are filled by the whole block: pulled from
// staging over PCIe (O_RDONLY) — or, for O_GWRONCE, left FILLING with
// sc.fill[i] = 1 for the caller (gwrite) to zero-fill/write. Busy pages are
// retried after the block's own fills, so no block waits on another while it
// holds an unfilled frame. Returns 0 with every sc.frame[i] held, or -errno
// with none held.
template <class G = BlockGroup>
__device__ int acquire_batch(const gfs_ctx* c, Scratch& sc, const FileSnap& fs, uint64_t pb, uint32_t cnt,
                             bool first_done) {
  const int tid = G::tid(), nthr = G::nthr();
  const bool fast = !(c->flags & GFS_F_LOCKED_TRAVERSAL);
  if (!first_done && tid < (int)cnt) sc.frame[tid] = kBusy;
  const uint64_t t0 = now_ns();
  uint32_t ns = 128;
  for (int round = 0;; ++round) {
    if (!(first_done && round == 0)) {
      if (tid < (int)cnt && sc.frame[tid] == kBusy) {
        // Retries of busy pages always try the lock-free path first: in the
        // locked ablation, hundreds of lanes re-taking the file lock while
        // they wait starve the lanes that still have to install pages.
        int f = (fast || round > 0) ? lookup_fast(c, fs, pb + tid, sc.lc_ok ? sc.leaf : nullptr) : -1;
        if (f < 0 && round > 0 && peek_busy(c, fs, pb + tid)) {
          // still being filled/evicted elsewhere: look again later without
          // taking the lock (lock-taking retries starve the installers)
        } else if (f >= 0) {
          sc.frame[tid] = f;
          sc.fill[tid] = 0;
          sc.stage[tid] = -1;
        } else {
          const Lk r = lookup_try(c, fs, pb + tid);
          sc.frame[tid] = r.frame;
          sc.fill[tid] = r.fill;
          sc.stage[tid] = r.stage;
          sc.nbytes[tid] = r.nbytes;
        }
      }
      G::sync();
    }
    int err = 0;
    bool busy = false, pull = false;
    for (uint32_t i = 0; i < cnt; ++i) {
      const int f = sc.frame[i];
      if (f == kBusy) busy = true;
      else if (f < 0) err = f;
      else if (sc.fill[i] && sc.stage[i] != -1) pull = true;
    }
    if (pull) {  // fill the frames this block installed: staging -> frame over PCIe, or peer frame -> frame
      for (uint32_t i = 0; i < cnt; ++i)
        if (sc.frame[i] >= 0 && sc.fill[i] && sc.stage[i] != -1) {
          block_copy_from_frame<true>(frame_ptr(c, (uint32_t)sc.frame[i]), fill_src(c, sc.stage[i], fs, pb + i),
                                      sc.nbytes[i], tid, nthr);
          // a writable page past the old EOF reads (and diffs) as zeros, not a previous tenant's bytes
          if ((fs.oflags & GFS_O_RDWR) && sc.nbytes[i] < c->page_size)
            block_zero(frame_ptr(c, (uint32_t)sc.frame[i]) + sc.nbytes[i], c->page_size - sc.nbytes[i], tid, nthr);
        }
      if (c->flags & GFS_F_EXPORTED) __threadfence_system();  // peers read our frames at system scope
      else __threadfence();
      G::sync();
      if (tid < (int)cnt && sc.frame[tid] >= 0 && sc.fill[tid] && sc.stage[tid] != -1) {
        const uint32_t f = (uint32_t)sc.frame[tid];
        fill_src_free(c, sc.stage[tid]);
        sc.stage[tid] = -1;
        sc.fill[tid] = 0;
        st_rlx(&c->f_valid[f], sc.nbytes[tid]);
        st_rlx(&c->f_hv[f], sc.nbytes[tid]);
        a64_and_rel(&c->f_state[f], fl64(GFS_ST_FILLING));  // publish the page
      }
    }
    if (err) {
      if (tid < (int)cnt && sc.frame[tid] >= 0) {
        const uint32_t f = (uint32_t)sc.frame[tid];
        if (sc.fill[tid]) frame_retire(c, f, GFS_ST_FILLING);  // an installed O_GWRONCE page nobody wrote
        frame_release(c, f);
      }
      G::sync();
      return err;
    }
    if (!busy) {
      if (pull) G::sync();
      return 0;
    }
    // still busy: back off and retry (the timeout decision is made by one
    // thread and broadcast, so every thread takes the same path)
    if (tid == 0) sc.busy = timed_out(c, t0) ? 1u : 0u;
    if (tid < 32) __nanosleep(ns);
    ns = ns < 2048 ? ns * 2 : 2048;
    G::sync();
    if (sc.busy) {
      if (tid == 0) ctr(c, GFS_C_TIMEOUT);
      if (tid < (int)cnt && sc.frame[tid] == kBusy) sc.frame[tid] = -ETIMEDOUT;  // error path next round
      G::sync();
    }
  }
}

// ------------------------------------------------------------------ read-ahead (NEXT-2)
// "read-ahead, data transfer scheduling, and asynchronous writes".
// A block whose gread continues where its previous gread on the same read-only
// file ended fetches the next c->readahead pages: each is installed (FILLING,
// no reference held) and its READ RPC posted, but nobody waits. The fill
// belongs to whoever completes it: the first lookup that needs the page takes
// it over in lookup_try (waits for the RPC, pulls the page, publishes it), and
// the issuing block reaps the ones nobody needed at its gclose. No lane ever
// waits for the issuing block itself, so read-ahead adds no wait-for edge
// between blocks (the host completes every RPC on its own).

// Post the read-ahead fetch of `page` (< the file's page count). Returns the
// frame, or -1 when the page is cached / in flight or no slot / frame is free.
__device__ __noinline__ int ra_issue(const gfs_ctx* c, const FileSnap& fs, uint64_t page, uint64_t* pv_out) {
  const int f0 = lookup_fast(c, fs, page, nullptr);
  if (f0 >= 0) {  // cached
    r64_add_rlx(&c->f_state[f0], kRefDec);
    return -1;
  }
  if (peek_busy(c, fs, page)) return -1;
  const uint64_t base = page << c->page_shift;
  const uint64_t rem = fs.size - base;
  const uint32_t nb = (uint32_t)(rem < c->page_size ? rem : c->page_size);
  const int st = stage_alloc(c, false);
  if (st < 0) return -1;
  uint64_t* slot = walk(c, fs.root, fs.height, page, true, nullptr);
  if (!slot) {
    stage_free(c, st);
    return -1;
  }
  const uint64_t s = ld_acq64(slot);
  if ((uint32_t)s) {  // only a stale slot (frame reassigned, or failed and not refilling) is replaced
    const uint64_t fst = ld_acq64(&c->f_state[slot_frame(s)]);
    const bool stale = (fst >> 32) != (s >> 32) ||
                       (((uint32_t)fst & GFS_ST_ERROR) && !((uint32_t)fst & GFS_ST_FILLING));
    if (!stale) {
      stage_free(c, st);
      return -1;
    }
  }
  uint32_t gen = 0;
  const int g = alloc_frame(c, ((uint64_t)fs.uid << 32) | (uint32_t)page, fs.fdx, &gen, true);
  if (g < 0) {
    stage_free(c, st);
    return -1;
  }
  st_rel64(&c->f_pf[g], GFS_PF_POSTING);  // lookups that find it now wait (busy) instead of adopting
  if (a64_cas(slot, s, slot_val_fill((uint32_t)g, gen)) != s) {
    st_rlx64(&c->f_pf[g], 0);
    frame_abandon(c, (uint32_t)g);
    stage_free(c, st);
    return -1;
  }
  a64_add_rel(&c->f_state[g], kRefDec);  // FILLING, unreferenced: the fill is anyone's to complete
  const int64_t t = rpc_post(c, GFS_OP_READ, fs.hfid, base, st, nb, 0, 0, nullptr, 0);
  if (t < 0) {  // not posted: the frame fails (a later lookup installs over it)
    st_rlx64(&c->f_pf[g], 0);
    stage_free(c, st);
    a64_or_rel(&c->f_state[g], GFS_ST_ERROR);
    a64_and_rel(&c->f_state[g], fl64(GFS_ST_FILLING));
    return -1;
  }
  const uint64_t pv = ((uint64_t)(t + 1) << 32) | (uint32_t)(st + 1);
  st_rel64(&c->f_pf[g], pv);
  *pv_out = pv;
  ctr(c, GFS_C_RA_ISSUED);
  ctr(c, GFS_C_MISS);
  ctr(c, GFS_C_RPC_READ);
  ctr(c, GFS_C_BYTES_H2D, nb);
  return g;
}

// After a block gread of [off, off + n) on read-only fd (warp 0 only): if it
// continued the block's previous gread on fd, post the fetches of the pages
// after it that are not fetched yet (up to c->readahead ahead), and forget
// the posted fills that other lookups completed meanwhile.
template <class G>
__device__ __noinline__ void ra_after(const gfs_ctx* c, Scratch& sc, const FileSnap& fs, int fd, uint64_t off,
                                      uint64_t n) {
  const int lane = block_tid() & 31;
  if (lane == 0 && (sc.ra_grid != grid_id() || sc.ra_blk != G::key())) {
    sc.ra_grid = grid_id();
    sc.ra_blk = G::key();
    sc.ra_fd = -1;
    sc.ra_n = 0;
    sc.ra_hi = 0;
    sc.ra_next = 0;
  }
  __syncwarp();
  const bool seq = sc.ra_fd == fd && sc.ra_next == off;
  const uint64_t p1 = (off + n - 1) >> c->page_shift;
  const uint64_t np = (fs.size + c->page_size - 1) >> c->page_shift;
  // keep the posted fills still pending (f_pf unchanged)
  const uint32_t n0 = sc.ra_n;
  bool keep = false;
  uint32_t kf = 0;
  uint64_t kv = 0;
  if ((uint32_t)lane < n0) {
    kf = sc.ra_f[lane];
    kv = sc.ra_v[lane];
    keep = ld_rlx64(&c->f_pf[kf]) == kv;
  }
  const uint32_t kb = __ballot_sync(0xFFFFFFFFu, keep);
  __syncwarp();
  if (keep) {
    const uint32_t k = __popc(kb & ((1u << lane) - 1u));
    sc.ra_f[k] = kf;
    sc.ra_v[k] = kv;
  }
  uint32_t nk = __popc(kb);
  uint64_t hi = seq ? sc.ra_hi : p1;
  if (seq) {
    const uint64_t lo = (sc.ra_hi > p1 ? sc.ra_hi : p1) + 1;
    uint64_t top = p1 + c->readahead;
    if (top > np - 1) top = np - 1;
    const uint64_t pg = lo + (uint64_t)lane;
    int g = -1;
    uint64_t pv = 0;
    if (lo <= top && pg <= top && nk + (uint32_t)lane < kRA) g = ra_issue(c, fs, pg, &pv);
    const uint32_t ib = __ballot_sync(0xFFFFFFFFu, g >= 0);
    __syncwarp();
    if (g >= 0) {
      const uint32_t k = nk + __popc(ib & ((1u << lane) - 1u));
      sc.ra_f[k] = (uint32_t)g;
      sc.ra_v[k] = pv;
    }
    nk += __popc(ib);
    if (lo <= top && top > hi) hi = top;
  }
  __syncwarp();
  if (lane == 0) {
    sc.ra_n = nk;
    sc.ra_fd = fd;
    sc.ra_next = off + n;
    sc.ra_hi = hi;
  }
  __syncwarp();
}

// At gclose (block-collective): complete every fill this block posted that is
// still pending — pull the page into its frame and publish it — so no frame
// stays FILLING and no staging or ring slot stays held after the block is gone.
template <class G>
__device__ __noinline__ void ra_reap(const gfs_ctx* c, Scratch& sc) {
  const int tid = G::tid(), nthr = G::nthr();
  if (!(sc.ra_grid == grid_id() && sc.ra_blk == G::key()) || sc.ra_n == 0) return;  // uniform: shared values
  const uint32_t n = sc.ra_n;
  if (tid < (int)n) {
    const uint32_t f = sc.ra_f[tid];
    const uint64_t v = sc.ra_v[tid];
    sc.frame[tid] = -1;
    if (a64_cas(&c->f_pf[f], v, 0) == v) {
      const int st = (int)(uint32_t)v - 1;
      const int32_t r = rpc_complete(c, (v >> 32) - 1, nullptr);
      if (r < 0) {
        stage_free(c, st);
        a64_or_rel(&c->f_state[f], GFS_ST_ERROR);
        a64_and_rel(&c->f_state[f], fl64(GFS_ST_FILLING));
      } else {
        sc.frame[tid] = (int)f;
        sc.stage[tid] = st;
        sc.nbytes[tid] = (uint32_t)r;
      }
    }
  }
  G::sync();
  for (uint32_t i = 0; i < n; ++i)
    if (sc.frame[i] >= 0)
      block_copy_from_frame<true>(frame_ptr(c, (uint32_t)sc.frame[i]), stage_ptr(c, sc.stage[i]), sc.nbytes[i], tid,
                                  nthr);
  if (c->flags & GFS_F_EXPORTED) __threadfence_system();
  else __threadfence();
  G::sync();
  if (tid < (int)n && sc.frame[tid] >= 0) {
    const uint32_t f = (uint32_t)sc.frame[tid];
    stage_free(c, sc.stage[tid]);
    st_rlx(&c->f_valid[f], sc.nbytes[tid]);
    st_rlx(&c->f_hv[f], sc.nbytes[tid]);
    st_rlx(&c->f_stamp[f], stamp_now());
    a64_and_rel(&c->f_state[f], fl64(GFS_ST_FILLING));  // publish: FILLING -> plain unreferenced page
    ctr(c, GFS_C_RA_REAPED);
  }
  if (tid == 0) {
    sc.ra_n = 0;
    sc.ra_fd = -1;
  }
  G::sync();
}

// O_RDWR write-back with the diff done on the GPU: for frame f
// and its pristine copy pf, bytes [lo, hi) of the page (lo a multiple of 64)
// go to staging slot `st` (working copy, at in-page offsets) and a bitmap to
// slot `mst`: bit j of 64-bit word w <=> byte lo + 64w + j differs. The host
// writes only those bytes (GFS_WF_MASK). PCIe carries 1 + 1/8 bytes per dirty
// byte instead of 2 (working + pristine). Block-collective.
__device__ __forceinline__ void diff_to_stage(const gfs_ctx* c, uint32_t f, uint32_t pf, uint32_t lo, uint32_t hi,
                                              int st, int mst, int tid, int nthr) {
  const uint8_t* w = frame_ptr(c, f) + lo;
  const uint8_t* p = frame_ptr(c, pf) + lo;
  uint8_t* out = stage_ptr(c, st) + lo;
  uint64_t* mask = (uint64_t*)stage_ptr(c, mst);
  const uint32_t nw = (hi - lo + 63) / 64;
  for (uint32_t k = tid; k < nw; k += nthr) {
    uint64_t m = 0;
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      const int4 a = __ldcg((const int4*)(w + 64 * k) + q), b = __ldcg((const int4*)(p + 64 * k) + q);
      ((int4*)(out + 64 * k))[q] = a;
      const uint32_t d[4] = {__vcmpne4(a.x, b.x), __vcmpne4(a.y, b.y), __vcmpne4(a.z, b.z), __vcmpne4(a.w, b.w)};
#pragma unroll
      for (int j = 0; j < 4; ++j)  // 0xFF/0x00 per byte -> 4 bits (as word_bits4 in the grep scan)
        m |= (uint64_t)((((d[j] >> 7) & 0x01010101u) * 0x00204081u) >> 21 & 0xFu) << (16 * q + 4 * j);
    }
    const uint32_t end = lo + 64 * k + 64;
    if (end > hi) m &= (hi - (lo + 64 * k) >= 64) ? ~0ull : ((1ull << (hi - (lo + 64 * k))) - 1ull);
    mask[k] = m;
  }
}

// O_RDWR: before the first local write to a page, preserve its
// pristine copy. Block-collective over the held frames sc.frame[0, cnt): lane
// i claims the pristine slot of page i (CAS 0 -> PENDING), allocates a frame
// for it (held FILLING|1, so never evicted or found), the block copies the
// working page into it and the lane publishes it; a page whose pristine copy
// another block is making is waited for (that block only copies a frame it
// holds: it never waits on us). Returns 0 or -errno (then no claim is left).
template <class G = BlockGroup>
__device__ __noinline__ int ensure_pristine(const gfs_ctx* c, Scratch& sc, uint32_t fdx, uint32_t cnt) {
  const int tid = G::tid(), nthr = G::nthr();
  if (tid == 0) sc.err = 0;
  if (tid < (int)cnt) {
    const uint32_t f = (uint32_t)sc.frame[tid];
    sc.lo[tid] = GFS_DIRTY_NONE;  // pristine frame this lane must fill
    if (ld_acq(&c->f_pristine[f]) == 0 && atom_cas(&c->f_pristine[f], 0u, GFS_PRISTINE_PENDING) == 0u) {
      uint32_t gen = 0;
      const int pf = alloc_frame(c, GFS_TAG_NONE, fdx, &gen);
      if (pf < 0) {
        st_rel(&c->f_pristine[f], 0u);
        atomicMin(&sc.err, pf);
      } else {
        sc.lo[tid] = (uint32_t)pf;
      }
    }
  }
  G::sync();
  for (uint32_t i = 0; i < cnt; ++i)
    if (sc.lo[i] != GFS_DIRTY_NONE)
      block_copy_from_frame(frame_ptr(c, sc.lo[i]), frame_ptr(c, (uint32_t)sc.frame[i]), c->page_size, tid, nthr);
  __threadfence();
  G::sync();
  if (tid < (int)cnt) {
    const uint32_t f = (uint32_t)sc.frame[tid];
    if (sc.lo[tid] != GFS_DIRTY_NONE) {
      st_rel(&c->f_pristine[f], sc.lo[tid] + 1u);
    } else {
      uint32_t ns = 64;
      const uint64_t t0 = now_ns();
      uint32_t pv;
      while ((pv = ld_acq(&c->f_pristine[f])) == GFS_PRISTINE_PENDING) {
        backoff(ns);
        if (timed_out(c, t0)) {
          atomicMin(&sc.err, -ETIMEDOUT);
          break;
        }
      }
      if (pv == 0) atomicMin(&sc.err, -ENOMEM);  // its maker found no frame: never write without a pristine copy
    }
  }
  G::sync();
  return sc.err;
}

// ------------------------------------------------------------------ file table
// Path hash: an order-sensitive SUM of per-(position, byte) mixes, so a warp
// can hash a path in parallel (lane l takes bytes l, l+32, ...).
__device__ __forceinline__ uint64_t path_term(uint32_t i, uint32_t b) {
  uint64_t z = (((uint64_t)i << 8) | b) * 0x9E3779B97F4A7C15ull;
  z = (z ^ (z >> 29)) * 0xBF58476D1CE4E5B9ull;
  return z ^ (z >> 32);
}
__device__ __forceinline__ uint64_t path_final(uint64_t sum, uint32_t n) {
  uint64_t z = sum ^ ((uint64_t)n * 0x94D049BB133111EBull);
  z = (z ^ (z >> 31)) * 0xBF58476D1CE4E5B9ull;
  return z ^ (z >> 29);
}
// Length (GFS_MAX_PATH if no NUL within it) and hash of `p`, by one thread.
__device__ __forceinline__ uint32_t path_len_hash(const char* p, uint64_t* h) {
  uint32_t n = 0;
  uint64_t sum = 0;
  while (n < GFS_MAX_PATH && p[n]) {
    sum += path_term(n, (uint8_t)p[n]);
    ++n;
  }
  *h = path_final(sum, n);
  return n;
}
// The same, by a full warp: one aligned 32-byte window per step (coalesced,
// never crosses a page, so no read faults past the NUL), one ballot per step.
__device__ __forceinline__ uint32_t path_len_hash_warp(const char* p, uint64_t* h) {
  const int lane = block_tid() & 31;
  const int off0 = (int)((uintptr_t)p & 31);
  const unsigned char* a = (const unsigned char*)((uintptr_t)p & ~(uintptr_t)31);
  uint64_t sum = 0;
  uint32_t n = GFS_MAX_PATH;
  for (int base = 0; base < (int)GFS_MAX_PATH + off0; base += 32) {
    const int i = base + lane - off0;  // index in the path; < 0: before it
    const uint32_t b = (i >= 0 && i < (int)GFS_MAX_PATH) ? a[base + lane] : 1u;
    const uint32_t z = __ballot_sync(0xFFFFFFFFu, b == 0);
    const int lim = z ? base + (__ffs(z) - 1) - off0 : (int)GFS_MAX_PATH;  // bytes before the NUL
    if (i >= 0 && i < lim) sum += path_term((uint32_t)i, b);
    if (z) {
      n = (uint32_t)lim;
      break;
    }
  }
  for (int o = 16; o; o >>= 1) sum += __shfl_xor_sync(0xFFFFFFFFu, sum, o);
  *h = path_final(sum, n);
  return n;
}
__device__ __forceinline__ bool snap_fd(const gfs_ctx* c, int fd, FileSnap* s) {
  if (fd < 0 || (uint32_t)fd >= c->max_files) return false;
  const gfs_file* e = c->files + fd;
  const uint32_t sr = ld_acq(&e->sr);
  if ((sr >> 24) != GFS_FS_OPEN || (sr & 0xFFFFFF) == 0) return false;
  // relaxed (L2) loads: an entry can be re-incarnated by another SM while
  // this SM still holds an L1 line of it from earlier in the launch
  s->fdx = (uint32_t)fd;
  s->uid = ld_rlx(&e->uid);
  s->root = ld_rlx(&e->root);
  s->height = ld_rlx(&e->height);
  s->hfid = ld_rlx(&e->hfid);
  s->oflags = ld_rlx(&e->oflags);
  s->size = ld_rlx64((const uint64_t*)&e->size);
  return true;
}

// Snapshot for gread: read-only files this block opened are served from the
// block's cached snapshot (their entry cannot change while held open).
template <class G = BlockGroup>
__device__ __forceinline__ bool snap_fd_cached(const gfs_ctx* c, Scratch& sc, int fd, FileSnap* s) {
  if (sc.cached_fd == fd && sc.cached_blk == G::key() && sc.cached_grid == grid_id()) {
    *s = sc.cached;
    return true;
  }
  return snap_fd(c, fd, s);
}

// Claim page p's frame for write-back if it is dirty and unreferenced.
// Returns the frame (state EVICTING) or -1 (clean / absent), or -EBUSY.
__device__ int claim_dirty(const gfs_ctx* c, const FileSnap& fs, uint64_t p) {
  uint64_t* slot = walk(c, fs.root, fs.height, p, false, nullptr);
  if (!slot) return -1;
  const uint64_t s = ld_acq64(slot);
  if (!(uint32_t)s) return -1;
  const uint32_t f = slot_frame(s);
  const uint64_t want = ((uint64_t)fs.uid << 32) | (uint32_t)p;
  if (ld_acq64(&c->f_tag[f]) != want || ld_rlx(&c->f_lo[f]) == GFS_DIRTY_NONE) return -1;
  if (!claim_frame(&c->f_state[f], 0u))
    return (ld_acq64(&c->f_tag[f]) == want && ld_rlx(&c->f_lo[f]) != GFS_DIRTY_NONE) ? -EBUSY : -1;
  if (ld_acq64(&c->f_tag[f]) != want || ld_rlx(&c->f_lo[f]) == GFS_DIRTY_NONE) {
    a64_and_rel(&c->f_state[f], fl64(GFS_ST_EVICTING));
    return -1;
  }
  return (int)f;
}

// Write back every dirty, unreferenced page of the snapshot file in [pb, pe)
// from a single thread (used by the re-open path). Returns 0, -EBUSY (a dirty
// page was mapped or in use, Tab.1), or a negative RPC error.
__device__ int sync_pages_lane(const gfs_ctx* c, const FileSnap& fs, uint64_t pb, uint64_t pe) {
  int rc = 0;
  for (uint64_t p = pb; p < pe; ++p) {
    const int f = claim_dirty(c, fs, p);
    if (f == -EBUSY) {
      if (rc == 0) rc = -EBUSY;
      continue;
    }
    if (f < 0) continue;
    const int32_t r = frame_writeback_lane(c, (uint32_t)f, fs.hfid);
    if (r < 0) rc = r;
    a64_and_rel(&c->f_state[f], fl64(GFS_ST_EVICTING));
  }
  return rc;
}

// Drop cached pages [pb, pe) of the snapshot file (gftruncate).
__device__ int drop_pages(const gfs_ctx* c, const FileSnap& fs, uint64_t pb, uint64_t pe, int tid, int nthr) {
  int rc = 0;
  for (uint64_t p = pb + tid; p < pe; p += nthr) {
    uint64_t* slot = walk(c, fs.root, fs.height, p, false, nullptr);
    if (!slot) continue;
    const uint64_t s = ld_acq64(slot);
    if (!(uint32_t)s) continue;
    const uint32_t f = slot_frame(s);
    const uint64_t want = ((uint64_t)fs.uid << 32) | (uint32_t)p;
    if (ld_acq64(&c->f_tag[f]) != want) continue;
    if (!claim_frame(&c->f_state[f], 0u)) {
      rc = -EBUSY;
      continue;
    }
    if (ld_acq64(&c->f_tag[f]) == want) {
      st_rlx(&c->f_lo[f], GFS_DIRTY_NONE);
      st_rlx(&c->f_hi[f], 0);
      st_rlx(&c->f_written[f], 0);
      st_rlx(&c->f_hv[f], 0);
      pristine_free(c, f);
      frame_retire(c, f, GFS_ST_EVICTING);  // slots naming this generation go stale
    } else {
      a64_and_rel(&c->f_state[f], fl64(GFS_ST_EVICTING));
    }
  }
  return rc;
}

__device__ __forceinline__ bool same_path(const gfs_ctx* c, const gfs_file* e, uint32_t fdx, const char* path,
                                          uint32_t n, uint64_t h) {
  if (ld_rlx64(&e->path_hash) != h || ld_rlx(&e->path_len) != n) return false;
  const char* sp = c->paths + (size_t)fdx * GFS_MAX_PATH;  // 1 KiB aligned
  if ((((uintptr_t)path) & 7) == 0) {
    // 8-byte words, no early exit (the loads pipeline); an aligned word never
    // crosses a page, so reading the caller's word holding the NUL is safe
    const uint32_t nw = (n + 7) / 8;
    uint64_t diff = 0;
    for (uint32_t k = 0; k < nw; ++k) {
      uint64_t x = __ldcg((const unsigned long long*)sp + k) ^ ((const unsigned long long*)path)[k];
      if (k == nw - 1 && (n & 7)) x &= (1ull << (8 * (n & 7))) - 1;
      diff |= x;
    }
    return diff == 0;
  }
  for (uint32_t i = 0; i < n; ++i)
    if (__ldcg((const unsigned char*)sp + i) != (unsigned char)path[i]) return false;
  return true;
}

// Open RPC + install of a fresh incarnation. `e` is held in OPENING/REOPENING.
__device__ int open_rpc_fill(const gfs_ctx* c, gfs_file* e, uint32_t fdx, uint32_t flags, uint32_t old_hfid_plus1,
                             gfs_rpc_resp* rs, int stage = -1) {
  const char* sp = c->paths + (size_t)fdx * GFS_MAX_PATH;
  const int32_t r = rpc_call(c, GFS_OP_OPEN, 0, 0, stage, 0, flags, old_hfid_plus1, sp, e->path_len, rs);
  ctr(c, GFS_C_RPC_OPEN);
  if (r < 0) return r;
  if (rs->status < 0) return rs->status;
  return 0;
}

__device__ int new_incarnation(const gfs_ctx* c, gfs_file* e, uint32_t flags, const gfs_rpc_resp& rs) {
  const uint32_t root = node_alloc(c);
  if (!root) return -ENOMEM;
  const uint64_t P = c->page_size;
  const uint64_t npages = ((uint64_t)rs.size + P - 1) >> c->page_shift;
  e->root = root;
  e->height = (flags & GFS_O_WRITABLE) ? GFS_MAX_HEIGHT : height_for(npages);  // writable files grow
  e->uid = atomicAdd(c->uid_next, 1u);
  e->hfid = rs.hfid;
  e->size = (uint64_t)rs.size;
  e->version = rs.version;
  e->ino = rs.ino;
  e->dev = rs.dev;
  e->mtime_ns = rs.mtime_ns;
  e->oflags = flags;
  e->synced_version = 0;
  e->zc = (flags & GFS_O_WRITABLE) ? 0ull : rs.pad[1];  // zero-copy source for read-only opens
  return 0;
}

// Move a file entry from state `from` to `to` (and adjust its count by dref)
// with one atomic delta, preserving transient increments of other openers.
__device__ __forceinline__ void sr_shift(gfs_file* e, uint32_t from, uint32_t to, int dref) {
  atom_add_rel(&e->sr, (uint32_t)(((to - from) << 24) + (uint32_t)dref));
}

// Page 0 fetched with the OPEN reply (GFS_O_PREFETCH): installed FILLING|1,
// the calling block pulls it from `stage` and publishes it.
struct Prefetch {
  int frame;
  int stage;
  uint32_t nbytes;
};

// gopen body, run by one thread.
// `n`, `h`: the path's length and hash (path_len_hash*).
__device__ int open_leader(const gfs_ctx* c, const char* path, uint32_t n, uint64_t h, int flags_in,
                           Prefetch* pf) {
  pf->frame = -1;
  pf->stage = -1;
  const bool want_pf = (flags_in & (int)GFS_O_PREFETCH) != 0;
  const int flags = flags_in & ~(int)GFS_O_PREFETCH;
  if (flags != (int)GFS_O_RDONLY && flags != (int)GFS_O_GWRONCE && flags != (int)GFS_O_RDWR) return -EINVAL;
  if (n == 0) return -ENOENT;
  if (n >= GFS_MAX_PATH) return -ENAMETOOLONG;
  const uint32_t mask = c->max_files - 1;
  uint32_t i = (uint32_t)h & mask;
  uint32_t probes = 0;
  const uint64_t t0 = now_ns();
  uint32_t ns = 64;
  for (;;) {
    if (probes > c->max_files) return -EMFILE;
    gfs_file* e = c->files + i;
    const uint32_t sr = ld_acq(&e->sr);
    const uint32_t st = sr >> 24;
    if (st == GFS_FS_FREE) {
      if (atom_cas(&e->sr, 0u, (GFS_FS_CLAIM << 24) | 1u) != 0u) continue;
      char* sp = c->paths + (size_t)i * GFS_MAX_PATH;
      for (uint32_t k = 0; k < n; ++k) sp[k] = path[k];
      sp[n] = 0;
      e->path_len = n;
      e->path_hash = h;
      e->lock = 0;
      e->err = 0;
      // From here on other openers may hold transient +1s on `sr` (fast path
      // below): every state change is an atomic delta, never a plain store.
      sr_shift(e, GFS_FS_CLAIM, GFS_FS_OPENING, 0);
      gfs_rpc_resp rs;
      // page-0 prefetch only if a staging slot is free right now (never wait
      // while the entry is OPENING: other openers of the file wait on it)
      const int pst = (want_pf && flags == (int)GFS_O_RDONLY) ? stage_alloc(c, false) : -1;
      int r = open_rpc_fill(c, e, i, (uint32_t)flags, 0, &rs, pst);
      if (r == 0) r = new_incarnation(c, e, (uint32_t)flags, rs);
      if (r < 0) {
        if (pst >= 0) stage_free(c, pst);
        e->err = r;
        sr_shift(e, GFS_FS_OPENING, GFS_FS_DEAD, -1);  // tombstone; a later gopen retries further along
        return r;
      }
      if (pst >= 0) {  // install page 0 while nobody else can see the file
        int ok = 0;
        const uint32_t nb = (uint32_t)rs.pad[0];
        uint64_t* slot = nb ? walk(c, e->root, e->height, 0, true, nullptr) : nullptr;
        if (slot) {
          uint32_t gen = 0;
          const int g = alloc_frame(c, (uint64_t)e->uid << 32, i, &gen);
          if (g >= 0) {
            if (a64_cas(slot, 0ull, detail::slot_val_fill((uint32_t)g, gen)) == 0ull) {
              pf->frame = g;
              pf->stage = pst;
              pf->nbytes = nb;
              ok = 1;
              ctr(c, GFS_C_MISS);
              ctr(c, GFS_C_BYTES_H2D, nb);
            } else {
              frame_abandon(c, (uint32_t)g);
            }
          }
        }
        if (!ok) stage_free(c, pst);
      }
      sr_shift(e, GFS_FS_OPENING, GFS_FS_OPEN, 0);
      return (int)i;
    }
    if (st == GFS_FS_CLAIM) {  // being inserted: wait for its path
      backoff(ns);
      if (timed_out(c, t0)) return -ETIMEDOUT;
      continue;
    }
    if (!same_path(c, e, i, path, n, h)) {
      i = (i + 1) & mask;
      ++probes;
      continue;
    }
    if (st == GFS_FS_DEAD) {
      i = (i + 1) & mask;
      ++probes;
      continue;
    }
    if (st == GFS_FS_OPENING || st == GFS_FS_REOPENING) {
      backoff(ns);
      if (timed_out(c, t0)) return -ETIMEDOUT;
      continue;
    }
    if (st == GFS_FS_OPEN) {
      if (ld_rlx(&e->oflags) != (uint32_t)flags) return -EBUSY;  // one writer at a time
      // Fast path: a plain increment, no CAS loop — hundreds of
      // blocks open the same file at once. Undo if the state moved meanwhile.
      const uint32_t old = atom_add_acq(&e->sr, 1u);
      if ((old >> 24) == GFS_FS_OPEN) {
        ctr(c, GFS_C_OPEN_FAST);  // no CPU communication
        return (int)i;
      }
      atom_add_rel(&e->sr, 0xFFFFFFFFu);
      continue;
    }
    if (st == GFS_FS_CLOSED) {
      if ((sr & 0xFFFFFF) != 0 || atom_cas(&e->sr, sr, (GFS_FS_REOPENING << 24) | 1u) != sr) {
        backoff(ns);
        continue;
      }
      // Closed-file cache: re-open validates against the host (lazy
      // invalidation). O_GWRONCE or a mode change always starts
      // a fresh incarnation (pristine copy = zeros).
      FileSnap old;
      old.fdx = i; old.uid = e->uid; old.root = e->root; old.height = e->height;
      old.hfid = e->hfid; old.oflags = e->oflags; old.size = e->size;
      if (old.oflags & GFS_O_WRITABLE) {  // never lose written data: sync before dropping
        const uint64_t np = (old.size + c->page_size - 1) >> c->page_shift;
        int r = sync_pages_lane(c, old, 0, np);
        if (r < 0 && r != -EBUSY) {
          sr_shift(e, GFS_FS_REOPENING, GFS_FS_CLOSED, -1);
          return r;
        }
      }
      gfs_rpc_resp rs;
      int r = open_rpc_fill(c, e, i, (uint32_t)flags, old.hfid + 1u, &rs);
      if (r < 0) {
        sr_shift(e, GFS_FS_REOPENING, GFS_FS_CLOSED, -1);
        return r;
      }
      const bool same = (uint32_t)flags == GFS_O_RDONLY && old.oflags == GFS_O_RDONLY &&
                        rs.version == e->version && (uint64_t)rs.size == e->size && rs.ino == e->ino &&
                        rs.dev == e->dev && rs.mtime_ns == e->mtime_ns;
      if (same) {
        e->hfid = rs.hfid;
        e->zc = rs.pad[1];
        ctr(c, GFS_C_REOPEN_VALID);
      } else {
        tree_free(c, old.root, old.height);  // old frames become orphans (tier 0)
        r = new_incarnation(c, e, (uint32_t)flags, rs);
        ctr(c, GFS_C_INVALIDATE);
        if (r < 0) {
          e->err = r;
          sr_shift(e, GFS_FS_REOPENING, GFS_FS_DEAD, -1);
          return r;
        }
      }
      sr_shift(e, GFS_FS_REOPENING, GFS_FS_OPEN, 0);
      return (int)i;
    }
    i = (i + 1) & mask;  // unknown state: skip
    ++probes;
  }
}

// gclose body: decrement; the holder that drops the count to zero moves the
// entry to the closed-file table unless it was re-opened meanwhile.
__device__ int close_leader(const gfs_ctx* c, int fd) {
  if (fd < 0 || (uint32_t)fd >= c->max_files) return -EBADF;
  gfs_file* e = c->files + fd;
  const uint32_t old = atom_add_rel(&e->sr, 0xFFFFFFFFu);
  if ((old >> 24) != GFS_FS_OPEN || (old & 0xFFFFFF) == 0) {
    atom_add_rel(&e->sr, 1u);
    return -EBADF;
  }
  if ((old & 0xFFFFFF) == 1) atom_cas(&e->sr, GFS_FS_OPEN << 24, GFS_FS_CLOSED << 24);
  return 0;  // no write-back
}

// Snapshot for a caller that holds `fd` open through a gopen ordered before
// the call (so the entry cannot change meanwhile): relaxed L2 loads only. An
// acquire compiles to LDG.STRONG + CCTL.IVALL, which drops the SM's whole L1
// (e.g. a consumer's L1-cached lookup tables) on every call.
__device__ __forceinline__ bool snap_fd_rlx(const gfs_ctx* c, int fd, FileSnap* s) {
  if (fd < 0 || (uint32_t)fd >= c->max_files) return false;
  const gfs_file* e = c->files + fd;
  // all loads issued together (one L2 round trip); the state is checked after
  const uint32_t sr = ld_rlx(&e->sr);
  s->fdx = (uint32_t)fd;
  s->uid = ld_rlx(&e->uid);
  s->root = ld_rlx(&e->root);
  s->height = ld_rlx(&e->height);
  s->hfid = ld_rlx(&e->hfid);
  s->oflags = ld_rlx(&e->oflags);
  s->size = ld_rlx64((const uint64_t*)&e->size);
  return (sr >> 24) == GFS_FS_OPEN && (sr & 0xFFFFFF) != 0;
}

// The head and tail bytes of one co-aligned span that tma_span() leaves out,
// copied by the calling thread alone (L2 loads: the frame may be refilled).
__device__ __forceinline__ void lane_edges(uint8_t* dst, const uint8_t* src, uint32_t n) {
  const uint32_t h0 = (16u - ((uint32_t)(uintptr_t)src & 15u)) & 15u;
  const uint32_t head = h0 < n ? h0 : n;
  const uint32_t mid = (n - head) & ~15u;
  for (uint32_t i = 0; i < head; ++i) dst[i] = __ldcg(src + i);
  for (uint32_t i = head + mid; i < n; ++i) dst[i] = __ldcg(src + i);
}

}  // namespace
}  // namespace detail

// ===================================================================== API
using detail::Scratch;

// gopen: returns an fd shared by all openers of the path on this GPU.
// flags: GFS_O_RDONLY or GFS_O_GWRONCE, optionally | GFS_O_PREFETCH (hint:
// when the open goes to the host, page 0 comes back with the reply and the
// calling block installs it — one RPC instead of two for small files).
template <class G>
__device__ inline int gopen_t(const gfs_ctx* c, const char* path, int flags) {
  Scratch& sc = G::sc();
  const int tid = G::tid();
  G::sync();
  uint64_t ph = 0;
  uint32_t pn = 0;
  if (G::nthr() >= 32) {  // warp 0 measures and hashes the path together
    if (tid < 32) pn = detail::path_len_hash_warp(path, &ph);
  } else if (tid == 0) {
    pn = detail::path_len_hash(path, &ph);
  }
  if (tid == 0) {
    detail::Prefetch pf;
    const int fd = detail::open_leader(c, path, pn, ph, flags, &pf);
    sc.ret = fd;
    sc.frame[0] = pf.frame;
    sc.stage[0] = pf.stage;
    sc.nbytes[0] = pf.nbytes;
    sc.cached_fd = -1;
    if (fd >= 0 && detail::snap_fd(c, fd, &sc.cached) && !(sc.cached.oflags & GFS_O_WRITABLE)) {
      sc.cached_grid = detail::grid_id();
      sc.cached_blk = G::key();
      sc.cached_fd = fd;
      for (int i = 0; i < detail::kLeafCache; ++i) sc.leaf[i] = 0;
    }
    detail::ensure_mbar<G>(sc);
  }
  G::sync();
  if (sc.frame[0] >= 0) {  // pull the prefetched page 0 and publish it
    const uint32_t f = (uint32_t)sc.frame[0];
    detail::block_copy_from_frame<true>(detail::frame_ptr(c, f), detail::stage_ptr(c, sc.stage[0]), sc.nbytes[0],
                                        tid, G::nthr());
    if (c->flags & GFS_F_EXPORTED) __threadfence_system();
    else __threadfence();
    G::sync();
    if (tid == 0) {
      detail::stage_free(c, sc.stage[0]);
      detail::st_rlx(&c->f_valid[f], sc.nbytes[0]);
      detail::st_rlx(&c->f_hv[f], sc.nbytes[0]);
      detail::a64_and_rel(&c->f_state[f], detail::fl64(GFS_ST_FILLING));
      detail::frame_release(c, f);
      sc.frame[0] = -1;
    }
    G::sync();
  }
  return (int)sc.ret;
}

// gclose: drops this block's reference; never writes back.
template <class G>
__device__ inline int gclose_t(const gfs_ctx* c, int fd) {
  Scratch& sc = G::sc();
  G::sync();
  if constexpr (G::kBlock) {
    if (c->readahead) detail::ra_reap<G>(c, sc);  // the block's read-ahead fills nobody completed
  }
  if (G::tid() == 0) {
    if (sc.cached_fd == fd) sc.cached_fd = -1;
    if constexpr (G::kBlock) {  // an unconsumed gread hint on this file (it holds nothing)
      if (sc.hint_grid == detail::grid_id() && sc.hint_blk == G::key() && sc.hint_fd == fd) sc.hint_ok = 0;
    }
    sc.ret = detail::close_leader(c, fd);
  }
  G::sync();
  return (int)sc.ret;
}

template <class G>
__device__ inline int64_t gfstat_size_t(const gfs_ctx* c, int fd) {
  Scratch& sc = G::sc();
  G::sync();
  if (G::tid() == 0) {
    detail::FileSnap s;
    sc.ret = detail::snap_fd(c, fd, &s) ? (int64_t)s.size : -EBADF;
  }
  G::sync();
  return sc.ret;
}

// gread past its first barrier when the call is not a one-page shared-memory
// hit: the page batches (misses, multi-page spans, global destinations). Kept
// out of line so the hit path's registers are not shaped by this code.
template <class G>
__device__ __noinline__ int64_t gread_batches(const gfs_ctx* c, int64_t n, uint64_t off, void* dst) {
  using namespace detail;
  Scratch& sc = G::sc();
  const int tid = G::tid(), nthr = G::nthr();
  const uint32_t shift = c->page_shift;
  const uint64_t P = c->page_size;
  const uint32_t B = c->max_batch < (uint32_t)nthr ? c->max_batch : (uint32_t)nthr;
  const FileSnap fs = sc.fs;
  const uint64_t p0 = off >> shift, p1 = (off + (uint64_t)n - 1) >> shift;
  // TMA path: shared-memory destination co-aligned with the file offset
  // ((dst - off) % 16 == 0, so frame and destination agree mod 16): aligned
  // middles by TMA, the call's head and tail bytes by warp 0.
  const bool tma = __isShared(dst) && (((uintptr_t)dst - off) & 15) == 0;
  for (uint64_t pb = p0; pb <= p1; pb += B) {
    const uint32_t cnt = (uint32_t)((p1 - pb + 1) < B ? (p1 - pb + 1) : B);
    const int err = acquire_batch<G>(c, sc, fs, pb, cnt, pb == p0);
    if (err) return err;
    const uint64_t bs = pb == p0 ? (off & (P - 1)) : 0;
    const uint64_t be = pb + cnt - 1 == p1 ? ((off + (uint64_t)n - 1) & (P - 1)) + 1 : P;
    const uint64_t batch_bytes = ((uint64_t)cnt << shift) - bs - (P - be);
    if (tma && batch_bytes < (1u << 20)) {  // mbarrier tx-count limit
      const uint32_t ph = sc.mbar_phase;
      if (tid == 0) {
        asm volatile("fence.proxy.async.shared::cta;" ::: "memory");  // prior generic use of dst
        uint32_t tx = 0;
        for (uint32_t i = 0; i < cnt; ++i) {  // interior pages are whole and aligned: only the
          const uint64_t p = pb + i;          // call's first and last pages have edges
          const uint64_t s = p == p0 ? (off & (P - 1)) : 0;
          const uint64_t e = p == p1 ? ((off + (uint64_t)n - 1) & (P - 1)) + 1 : P;
          tx += span_mid(frame_ptr(c, (uint32_t)sc.frame[i]) + s, (uint32_t)(e - s));
        }
        mbar_expect_tx(&sc.mbar, tx);
        for (uint32_t i = 0; i < cnt; ++i) {
          const uint64_t p = pb + i;
          const uint64_t s = p == p0 ? (off & (P - 1)) : 0;
          const uint64_t e = p == p1 ? ((off + (uint64_t)n - 1) & (P - 1)) + 1 : P;
          tma_span((uint8_t*)dst + ((p << shift) + s - off), frame_ptr(c, (uint32_t)sc.frame[i]) + s,
                   (uint32_t)(e - s), &sc.mbar);
        }
      }
      if (tid < 32) {
        if (pb == p0) {
          const uint64_t s = off & (P - 1), e = p0 == p1 ? ((off + (uint64_t)n - 1) & (P - 1)) + 1 : P;
          copy_edges((uint8_t*)dst, frame_ptr(c, (uint32_t)sc.frame[0]) + s, (uint32_t)(e - s), tid);
        }
        if (pb + cnt - 1 == p1 && p1 != p0) {
          const uint64_t e = ((off + (uint64_t)n - 1) & (P - 1)) + 1;
          copy_edges((uint8_t*)dst + ((p1 << shift) - off), frame_ptr(c, (uint32_t)sc.frame[cnt - 1]), (uint32_t)e, tid);
        }
      }
      mbar_wait(&sc.mbar, ph);
      G::sync();
      if (tid == 0) sc.mbar_phase = ph ^ 1u;
    } else {
      for (uint32_t i = 0; i < cnt; ++i) {
        const uint64_t p = pb + i;
        const uint64_t s = p == p0 ? (off & (P - 1)) : 0;
        const uint64_t e = p == p1 ? ((off + (uint64_t)n - 1) & (P - 1)) + 1 : P;
        block_copy_from_frame((uint8_t*)dst + ((p << shift) + s - off), frame_ptr(c, (uint32_t)sc.frame[i]) + s,
                              e - s, tid, nthr);
      }
      G::sync();
    }
    if (tid < (int)cnt) frame_release(c, (uint32_t)sc.frame[tid]);
  }
  return n;
}

// gread: pread semantics; returns min(len, S-off) bytes, 0 at/after EOF.
template <class G, bool kHint = false>
__device__ inline int64_t gread_t(const gfs_ctx* c, int fd, uint64_t off, uint64_t len, void* dst,
                                  uint64_t next_off = ~0ull) {
  using namespace detail;
  Scratch& sc = G::sc();
  const int tid = G::tid(), nthr = G::nthr();
  const uint32_t shift = c->page_shift;
  const uint64_t P = c->page_size;
  const uint32_t B = c->max_batch < (uint32_t)nthr ? c->max_batch : (uint32_t)nthr;
  const bool fast = !(c->flags & GFS_F_LOCKED_TRAVERSAL);
  G::sync();  // the call is a barrier: earlier uses of dst by the block are complete
  // Warp 0 alone: snapshot + clip, then the first batch's fast-path lookups
  // (one page per lane). Other warps only touch `sc` after the next barrier.
  if (tid < 32) {
    if (tid == 0) {
      ensure_mbar<G>(sc);
      FileSnap s;
      const bool cached = sc.cached_fd == fd && sc.cached_blk == G::key() && sc.cached_grid == grid_id();
      if (cached) s = sc.cached;
      if (!(cached || snap_fd(c, fd, &s)) || (s.oflags & GFS_O_GWRONCE)) {
        sc.ret = -EBADF;
      } else {
        sc.fs = s;
        sc.lc_ok = cached ? 1u : 0u;
        sc.ret = off >= s.size ? 0 : (int64_t)(len < s.size - off ? len : s.size - off);
        ctr(c, GFS_C_GREAD_CALLS);
        if (sc.ret > 0) ctr(c, GFS_C_GREAD_BYTES, (unsigned long long)sc.ret);
      }
    }
    __syncwarp(nthr >= 32 ? 0xFFFFFFFFu : ((1u << nthr) - 1u));
    const int64_t n0 = sc.ret;
    uint32_t quick = 0;
    // the previous call's hint: the leaf slot of this call's first page, read
    // while that call's copy was in flight (0: none)
    uint64_t hsv = 0;
    if constexpr (G::kBlock && kHint) {
      if (tid == 0 && sc.hint_grid == grid_id() && sc.hint_blk == G::key() && sc.hint_ok) {
        if (n0 > 0 && sc.hint_fd == fd && sc.hint_page == (off >> shift)) hsv = sc.hint_sv;
        sc.hint_ok = 0;
      }
    }
    if (n0 > 0) {
      const uint64_t q0 = off >> shift, q1 = (off + (uint64_t)n0 - 1) >> shift;
      const uint32_t cnt = (uint32_t)((q1 - q0 + 1) < B ? (q1 - q0 + 1) : B);
      if (tid < (int)cnt) {
        const FileSnap fs0 = sc.fs;
        const bool quick_ok =
            q0 == q1 && n0 < (1 << 20) && __isShared(dst) && (((uintptr_t)dst - off) & 15) == 0;
        if (fast && quick_ok && !(c->flags & GFS_F_NO_SPECULATE)) {
          // Speculative one-page hit (lane 0; cnt == 1): a slot whose fill is known
          // complete (no kSlotFill) lets the copy start with the reference still in
          // flight. The reference's old state decides: same generation and no
          // FILLING / EVICTING / ERROR means the frame held this page's bytes from
          // the slot read on (a generation is never reused), so the copy is kept;
          // otherwise the reference is dropped, the copy waited out (it may not
          // land after dst is reused) and the call takes the normal path.
          // (a hinted slot value was read earlier: the same argument holds from
          // that read on, and a stale one fails the generation check)
          uint64_t* const sp = hsv ? nullptr : leaf_slot(c, fs0, q0, sc.lc_ok ? sc.leaf : nullptr);
          const uint64_t sv = hsv ? hsv : sp ? ld_rlx64(sp) : 0ull;
          if ((uint32_t)sv && !((uint32_t)sv & kSlotFill)) {
            const uint32_t fs_ = slot_frame(sv);
            const uint64_t old = a64_add_rlx(&c->f_state[fs_], 1ull);
            asm volatile("fence.proxy.async.shared::cta;" ::: "memory");  // prior generic use of dst
            uint64_t* mb = &sc.mbar;
            const uint8_t* src = frame_ptr(c, fs_) + (off & (P - 1));
            mbar_expect_tx(mb, span_mid(src, (uint32_t)n0));
            tma_span((uint8_t*)dst, src, (uint32_t)n0, mb);
            if ((old >> 32) == (sv >> 32) && !((uint32_t)old & (GFS_ST_FILLING | GFS_ST_EVICTING | GFS_ST_ERROR))) {
              ctr(c, GFS_C_HIT);
              ctr(c, GFS_C_LOCKFREE);
              sc.frame[0] = (int32_t)fs_;
              quick = 1;
            } else {
              r64_add_rlx(&c->f_state[fs_], kRefDec);
              mbar_wait(mb, sc.mbar_phase);
              sc.mbar_phase ^= 1u;
            }
          }
        }
        int f = quick ? -2 : fast ? lookup_fast(c, fs0, q0 + tid, sc.lc_ok ? sc.leaf : nullptr) : -1;
        if (quick) {
          // the speculative copy is in flight (above)
        } else if (f < 0) {
          const Lk r = lookup_try(c, fs0, q0 + tid);
          sc.frame[tid] = r.frame;
          sc.fill[tid] = r.fill;
          sc.stage[tid] = r.stage;
          sc.nbytes[tid] = r.nbytes;
        } else if (q0 == q1 && n0 < (1 << 20) && __isShared(dst) && (((uintptr_t)dst - off) & 15) == 0) {
          // Quick path: a one-page hit into shared memory. Lane 0 issues the
          // TMA bulk copy of the aligned middle now, before the block barrier,
          // so the copy overlaps the other warps' arrival; they only wait on
          // the mbarrier (head/tail bytes are copied by warp 0 after it).
          asm volatile("fence.proxy.async.shared::cta;" ::: "memory");  // prior generic use of dst
          uint64_t* mb = &sc.mbar;
          const uint8_t* src = frame_ptr(c, (uint32_t)f) + (off & (P - 1));
          mbar_expect_tx(mb, span_mid(src, (uint32_t)n0));
          tma_span((uint8_t*)dst, src, (uint32_t)n0, mb);
          sc.frame[0] = f;
          quick = 1;
        } else {
          sc.frame[tid] = f;
          sc.fill[tid] = 0;
          sc.stage[tid] = -1;
        }
      }
    }
    if (tid == 0) sc.quick = quick;
  }
  G::sync();
  const int64_t n = sc.ret;
  if (n <= 0) return n;
  int64_t res = n;
  if (sc.quick) {
    const uint32_t ph = sc.mbar_phase;
    copy_edges((uint8_t*)dst, frame_ptr(c, (uint32_t)sc.frame[0]) + (off & (P - 1)), (uint32_t)n, tid);
    if constexpr (G::kBlock && kHint) {
      // hint: read the leaf slot of the next call's first page while the copy
      // flies (no reference: the next call's speculative copy validates it)
      if (next_off != ~0ull && tid == 0 && fast && next_off < sc.fs.size) {
        sc.hint_grid = grid_id();
        sc.hint_blk = G::key();
        sc.hint_fd = fd;
        sc.hint_page = next_off >> shift;
        uint64_t* const nsp = leaf_slot(c, sc.fs, sc.hint_page, sc.lc_ok ? sc.leaf : nullptr);
        sc.hint_sv = nsp ? ld_rlx64(nsp) : 0ull;
        sc.hint_ok = sc.hint_sv != 0;
      }
    }
    mbar_wait(&sc.mbar, ph);
    G::sync();
    if (tid == 0) {
      sc.mbar_phase = ph ^ 1u;
      frame_release(c, (uint32_t)sc.frame[0]);
    }
  } else {
    res = gread_batches<G>(c, n, off, dst);
  }
  if constexpr (G::kBlock) {  // NEXT-2: read-ahead of a sequential reader of a read-only file (warp 0)
    if (c->readahead && res > 0 && tid < 32 && !(sc.fs.oflags & GFS_O_WRITABLE) && !c->npeers &&
        ld_rlx64(&c->files[sc.fs.fdx].zc) == 0)
      ra_after<G>(c, sc, sc.fs, fd, off, (uint64_t)res);
  }
  return res;
}

// Threadblock-collective calls (the prototype's granularity).
__device__ inline int gopen(const gfs_ctx* c, const char* path, int flags) {
  return gopen_t<detail::BlockGroup>(c, path, flags);
}
__device__ inline int gclose(const gfs_ctx* c, int fd) { return gclose_t<detail::BlockGroup>(c, fd); }
__device__ inline int64_t gfstat_size(const gfs_ctx* c, int fd) { return gfstat_size_t<detail::BlockGroup>(c, fd); }
__device__ inline int64_t gread(const gfs_ctx* c, int fd, uint64_t off, uint64_t len, void* dst) {
  return gread_t<detail::BlockGroup>(c, fd, off, len, dst);
}
// gread with the offset of the block's NEXT gread on the same file (a split-
// phase lookup, NEXT-2): while this call's one-page copy into
// shared memory is in flight, lane 0 reads the leaf slot of the page holding
// next_off (no reference is taken), so the next gread_hint starts its
// speculative copy right after its opening barrier, without a tree access;
// the copy is validated by the reference as always (a stale slot value fails
// the generation check and the call takes the normal path). A hint for
// another offset is ignored; next_off = ~0: no hint. Plain gread does not look
// at hints (it pays nothing for them).
__device__ inline int64_t gread_hint(const gfs_ctx* c, int fd, uint64_t off, uint64_t len, void* dst,
                                     uint64_t next_off) {
  return gread_t<detail::BlockGroup, true>(c, fd, off, len, dst, next_off);
}

// Warp-collective calls (the paper's design point): every lane of
// one warp calls with identical arguments; warps of a block proceed
// independently (no block barrier). Blocks using them have full warps and at
// most GFS_WARP_API_MAX_WARPS warps. Same semantics and errors as the block
// calls; `dst` may be global or shared memory.
__device__ inline int gopen_warp(const gfs_ctx* c, const char* path, int flags) {
  return gopen_t<detail::WarpGroup>(c, path, flags);
}
__device__ inline int gclose_warp(const gfs_ctx* c, int fd) { return gclose_t<detail::WarpGroup>(c, fd); }
__device__ inline int64_t gfstat_size_warp(const gfs_ctx* c, int fd) {
  return gfstat_size_t<detail::WarpGroup>(c, fd);
}
__device__ inline int64_t gread_warp(const gfs_ctx* c, int fd, uint64_t off, uint64_t len, void* dst) {
  return gread_t<detail::WarpGroup>(c, fd, off, len, dst);
}

namespace detail {
namespace {
// gread_lanes' one-request-at-a-time remainder, out of line so the callers'
// fast path keeps its registers.
__device__ __noinline__ int64_t gread_warp_slow(const gfs_ctx* c, int fd, uint64_t off, uint64_t len, void* dst) {
  return gread_t<WarpGroup>(c, fd, off, len, dst);
}
}  // namespace
}  // namespace detail

// gread_lanes: a warp-collective VECTORED gread (an extension in the spirit of
// P:L449-452's "data transfer scheduling"): every lane of the calling warp
// passes its OWN request (fd, off, len, dst) and receives its own result, with
// gread's pread semantics (EOF at the size snapshot). A
// lane passing len 0 (or fd < 0) takes no part and gets 0 (-EBADF for a bad
// fd with len > 0).
//
// Requests whose span covers at most two pages that are all cache hits, and
// whose destination is shared memory co-aligned with the offset
// ((dst - off) % 16 == 0), are served in one round: the lanes look their pages
// up at the same time (lock-free, one atomic per page), lane 0
// arms the warp's mbarrier with the total byte count, every lane issues its
// own TMA bulk copies (cp.async.bulk) and copies its <16-byte edges, and the
// warp waits ONCE for all of them — 32 requests cost about one request's
// latency. Every other request (a miss, a longer span, a global destination)
// is served one at a time by gread_warp, so misses keep their full semantics
// (RPC, eviction). Each fd must be held open by the caller through a gopen
// ordered before the call (the snapshot uses relaxed loads only, so the SM's
// L1 survives the call). Full warps only; uses the warp's scratch.
//
// Split phase (NEXT-2): gread_lanes_issue() returns once the hit
// copies are IN FLIGHT (misses and other requests are complete by then);
// gread_lanes_wait() waits for them and drops the page references. The
// destination must not be touched in between; a warp has at most one issued,
// unwaited request set, and makes no other warp-API call until it waits.
// gread_lanes(...) is issue + wait.
struct GreadLaneTicket {
  int64_t ret;     // the lane's result
  int32_t f0, f1;  // frames this lane holds until the wait (-1: none)
  uint32_t total;  // (warp-uniform) bytes in flight on the warp's mbarrier; 0: nothing to wait for
  uint32_t phase;  // (warp-uniform) the mbarrier phase to wait for
};

__device__ inline GreadLaneTicket gread_lanes_issue(const gfs_ctx* c, int fd, uint64_t off, uint64_t len,
                                                    void* dst) {
  using namespace detail;
  Scratch& sc = WarpGroup::sc();
  const int lane = block_tid() & 31;
  const uint32_t shift = c->page_shift;
  const uint64_t P = c->page_size;
  __syncwarp();
  GreadLaneTicket t{0, -1, -1, 0, 0};
  FileSnap s;
  if (len > 0 && fd >= 0) {
    if (!snap_fd_rlx(c, fd, &s) || (s.oflags & GFS_O_GWRONCE)) t.ret = -EBADF;
    else t.ret = off >= s.size ? 0 : (int64_t)(len < s.size - off ? len : s.size - off);
  } else if (len > 0) {
    t.ret = -EBADF;
  }
  uint32_t tx = 0, n0 = 0;
  if (t.ret > 0 && t.ret < (1 << 20) && !(c->flags & GFS_F_LOCKED_TRAVERSAL) && __isShared(dst) &&
      (((uintptr_t)dst - off) & 15) == 0) {
    const uint64_t p0 = off >> shift, p1 = (off + (uint64_t)t.ret - 1) >> shift;
    if (p1 - p0 <= 1) {
      t.f0 = lookup_fast(c, s, p0, nullptr);
      if (t.f0 >= 0 && p1 != p0) {
        t.f1 = lookup_fast(c, s, p1, nullptr);
        if (t.f1 < 0) {
          r64_add_rlx(&c->f_state[t.f0], kRefDec);
          t.f0 = -1;
        }
      }
      if (t.f0 >= 0) {
        const uint64_t in0 = off & (P - 1);
        n0 = (uint32_t)(t.f1 >= 0 ? P - in0 : (uint64_t)t.ret);
        tx = span_mid(frame_ptr(c, (uint32_t)t.f0) + in0, n0);
        if (t.f1 >= 0) tx += span_mid(frame_ptr(c, (uint32_t)t.f1), (uint32_t)t.ret - n0);
      }
    }
  }
  const bool fast = t.f0 >= 0;
  // the other requests first, one at a time, with the full warp-collective
  // gread (it completes its own mbarrier phases before the fast copies arm one)
  uint32_t slow = __ballot_sync(0xFFFFFFFFu, t.ret > 0 && !fast);
  while (slow) {
    const int src = __ffs(slow) - 1;
    slow &= slow - 1;
    const int sfd = __shfl_sync(0xFFFFFFFFu, fd, src);
    const uint64_t soff = __shfl_sync(0xFFFFFFFFu, off, src);
    const uint64_t slen = __shfl_sync(0xFFFFFFFFu, len, src);
    void* sdst = (void*)__shfl_sync(0xFFFFFFFFu, (unsigned long long)(uintptr_t)dst, src);
    const int64_t r = detail::gread_warp_slow(c, sfd, soff, slen, sdst);
    if (lane == src) t.ret = r;
  }
  t.total = __reduce_add_sync(0xFFFFFFFFu, tx);
  if (lane == 0) {
    ensure_mbar<WarpGroup>(sc);
    if (t.total) mbar_expect_tx(&sc.mbar, t.total);  // armed before any copy is issued
  }
  __syncwarp();
  t.phase = sc.mbar_phase;
  if (fast) {
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");  // earlier generic use of dst
    const uint8_t* s0 = frame_ptr(c, (uint32_t)t.f0) + (off & (P - 1));
    tma_span((uint8_t*)dst, s0, n0, &sc.mbar);
    lane_edges((uint8_t*)dst, s0, n0);
    if (t.f1 >= 0) {
      const uint8_t* s1 = frame_ptr(c, (uint32_t)t.f1);
      tma_span((uint8_t*)dst + n0, s1, (uint32_t)t.ret - n0, &sc.mbar);
      lane_edges((uint8_t*)dst + n0, s1, (uint32_t)t.ret - n0);
    }
  }
  __syncwarp();
  if (lane == 0 && t.total) sc.mbar_phase = t.phase ^ 1u;  // this phase belongs to the ticket now
  const uint32_t nfast = __popc(__ballot_sync(0xFFFFFFFFu, fast));
  const uint32_t bfast = __reduce_add_sync(0xFFFFFFFFu, fast ? (uint32_t)t.ret : 0u);
  if (lane == 0 && nfast) {
    ctr(c, GFS_C_GREAD_CALLS, nfast);
    ctr(c, GFS_C_GREAD_BYTES, bfast);
  }
  return t;
}

__device__ inline int64_t gread_lanes_wait(const gfs_ctx* c, GreadLaneTicket& t) {
  using namespace detail;
  Scratch& sc = WarpGroup::sc();
  if (t.total) mbar_wait(&sc.mbar, t.phase);
  __syncwarp();
  if (t.f0 >= 0) frame_release(c, (uint32_t)t.f0);
  if (t.f1 >= 0) frame_release(c, (uint32_t)t.f1);
  t.f0 = t.f1 = -1;
  t.total = 0;
  return t.ret;
}

__device__ inline int64_t gread_lanes(const gfs_ctx* c, int fd, uint64_t off, uint64_t len, void* dst) {
  GreadLaneTicket t = gread_lanes_issue(c, fd, off, len, dst);
  return gread_lanes_wait(c, t);
}

// gwrite: pwrite semantics on an O_GWRONCE file.
// New pages are zero-filled (never fetched); the dirty range and written byte
// count are kept per frame; a fence makes the data visible to write-back
// (P:L577-582).
__device__ inline int64_t gwrite(const gfs_ctx* c, int fd, uint64_t off, uint64_t len, const void* src) {
  using namespace detail;
  Scratch& sc = scratch();
  const int tid = block_tid(), nthr = block_nthr();
  __syncthreads();
  if (tid == 0) {
    FileSnap s;
    if (!snap_fd(c, fd, &s) || !(s.oflags & GFS_O_WRITABLE)) {
      sc.ret = -EBADF;
    } else if (off + len < off || ((off + len) >> c->page_shift) >= (1ull << 32)) {
      sc.ret = -EINVAL;
    } else {
      sc.fs = s;
      sc.lc_ok = 0;
      sc.ret = (int64_t)len;
      ctr(c, GFS_C_GWRITE_CALLS);
    }
  }
  __syncthreads();
  const int64_t n = sc.ret;
  if (n <= 0) return n;
  const FileSnap fs = sc.fs;
  const uint32_t shift = c->page_shift;
  const uint64_t P = c->page_size;
  const uint64_t p0 = off >> shift, p1 = (off + (uint64_t)n - 1) >> shift;
  const uint32_t B = c->max_batch < (uint32_t)nthr ? c->max_batch : (uint32_t)nthr;
  for (uint64_t pb = p0; pb <= p1; pb += B) {
    const uint32_t cnt = (uint32_t)((p1 - pb + 1) < B ? (p1 - pb + 1) : B);
    const int err = acquire_batch(c, sc, fs, pb, cnt, false);
    if (err) return err;
    if (fs.oflags & GFS_O_RDWR) {
      // pages past the host EOF start as zeros; then every page keeps its
      // pristine copy before the first local write (diff-and-merge)
      for (uint32_t i = 0; i < cnt; ++i)
        if (sc.fill[i]) block_zero(frame_ptr(c, (uint32_t)sc.frame[i]), P, tid, nthr);
      __syncthreads();
      const int perr = ensure_pristine(c, sc, fs.fdx, cnt);
      if (perr) {
        if (tid < (int)cnt) {
          const uint32_t f = (uint32_t)sc.frame[tid];
          if (sc.fill[tid]) frame_retire(c, f, GFS_ST_FILLING);
          frame_release(c, f);
        }
        __syncthreads();
        return perr;
      }
    }
    for (uint32_t i = 0; i < cnt; ++i) {
      const uint64_t p = pb + i;
      const uint64_t s = p == p0 ? (off & (P - 1)) : 0;
      const uint64_t e = p == p1 ? ((off + (uint64_t)n - 1) & (P - 1)) + 1 : P;
      uint8_t* fp = frame_ptr(c, (uint32_t)sc.frame[i]);
      if (sc.fill[i] && !(fs.oflags & GFS_O_RDWR)) {  // pristine copy is zeros
        block_zero(fp, s, tid, nthr);
        block_zero(fp + e, P - e, tid, nthr);
      }
      block_copy_plain(fp + s, (const uint8_t*)src + ((p << shift) + s - off), e - s, tid, nthr);
    }
    __threadfence();
    __syncthreads();
    if (tid < (int)cnt) {
      const uint32_t f = (uint32_t)sc.frame[tid];
      const uint64_t p = pb + tid;
      const uint32_t s = (uint32_t)(p == p0 ? (off & (P - 1)) : 0);
      const uint32_t e = (uint32_t)(p == p1 ? ((off + (uint64_t)n - 1) & (P - 1)) + 1 : P);
      atomicMin(&c->f_lo[f], s);
      atomicMax(&c->f_hi[f], e);
      atomicAdd(&c->f_written[f], e - s);
      if (sc.fill[tid]) a64_and_rel(&c->f_state[f], fl64(GFS_ST_FILLING));
      frame_release_rel(c, f);
    }
  }
  if (tid == 0) atomicMax((unsigned long long*)&c->files[fd].size, (unsigned long long)(off + (uint64_t)n));
  __syncthreads();
  return n;
}

// gfsync: synchronously write back all dirty pages of the file that are not
// mapped or in use (Tab.1); on success the data is in the host page
// cache. Block-cooperative: warp-0 lanes claim up to 32 dirty
// pages, the block copies their dirty ranges into staging slots over PCIe,
// then the lanes post the WRITE RPCs in parallel. Returns -EBUSY if busy
// dirty pages were skipped.
__device__ inline int gfsync(const gfs_ctx* c, int fd) {
  using namespace detail;
  Scratch& sc = scratch();
  const int tid = block_tid(), nthr = block_nthr();
  __syncthreads();
  if (tid == 0) {
    FileSnap s;
    if (!snap_fd(c, fd, &s)) {
      sc.ret = -EBADF;
    } else {
      sc.fs = s;
      sc.ret = 0;
      sc.err = 0;
    }
  }
  __syncthreads();
  if (sc.ret < 0) return (int)sc.ret;
  const FileSnap fs = sc.fs;
  if (fs.oflags & GFS_O_WRITABLE) {
    const uint64_t np = (fs.size + c->page_size - 1) >> c->page_shift;
    const uint32_t B = nthr < 32 ? (uint32_t)nthr : 32u;
    uint32_t ns = 256;
    const uint64_t t0 = now_ns();
    // Blocks syncing one file together start at different batches (rotated by
    // block id) so the dirty pages spread over them instead of the first
    // blocks claiming most of them; every block still visits every batch.
    const uint64_t nbat = (np + B - 1) / B;
    const uint64_t b0 = nbat ? block_linear() % nbat : 0;
    for (uint64_t bi = 0; bi < nbat;) {
      const uint64_t pb = ((b0 + bi) % nbat) * B;
      const uint32_t cnt = (uint32_t)((np - pb) < B ? (np - pb) : B);
      if (tid == 0) sc.busy = 0;
      __syncthreads();
      if (tid < (int)cnt) {
        const int f = claim_dirty(c, fs, pb + tid);
        sc.frame[tid] = f;
        sc.stage[tid] = -1;
        if (f == -EBUSY) atomicMin(&sc.err, -EBUSY);
        if (f >= 0) {
          sc.lo[tid] = ld_rlx(&c->f_lo[f]);
          sc.hi[tid] = ld_rlx(&c->f_hi[f]);
          const uint32_t pv = ld_rlx(&c->f_pristine[f]);
          sc.nbytes[tid] = (pv != 0 && pv != GFS_PRISTINE_PENDING) ? pv : 0u;  // O_RDWR: pristine frame + 1
          // no waiting for a staging slot while holding a claimed page (other
          // blocks may hold the slots and wait for pages): give the claim
          // back and redo this batch after the others are written. An O_RDWR
          // page needs two slots (working and pristine ranges, GFS_WF_DIFF).
          int st = stage_alloc(c, false), st2 = -1;
          if (st >= 0 && sc.nbytes[tid]) {
            st2 = stage_alloc(c, false);
            if (st2 < 0) {
              stage_free(c, st);
              st = -1;
            }
          }
          sc.stage[tid] = st;
          sc.fill[tid] = (uint32_t)st2;
          if (st < 0) {
            a64_and_rel(&c->f_state[f], fl64(GFS_ST_EVICTING));
            sc.frame[tid] = -1;
            sc.busy = 1;
          }
        }
      }
      __syncthreads();
      for (uint32_t i = 0; i < cnt; ++i)
        if (sc.frame[i] >= 0) {
          if (sc.nbytes[i]) {  // O_RDWR: the GPU diffs; the host gets the working bytes + a changed-byte mask
            diff_to_stage(c, (uint32_t)sc.frame[i], sc.nbytes[i] - 1, sc.lo[i] & ~63u, sc.hi[i], sc.stage[i],
                          (int)sc.fill[i], tid, nthr);
          } else {
            block_copy_from_frame(stage_ptr(c, sc.stage[i]) + sc.lo[i],
                                  frame_ptr(c, (uint32_t)sc.frame[i]) + sc.lo[i], sc.hi[i] - sc.lo[i], tid, nthr);
          }
        }
      __threadfence_system();
      __syncthreads();
      if (tid < (int)cnt && sc.frame[tid] >= 0) {
        const uint32_t f = (uint32_t)sc.frame[tid];
        const uint32_t lo = sc.lo[tid], hi = sc.hi[tid];
        const uint32_t wr = ld_rlx(&c->f_written[f]);
        const bool diff = sc.nbytes[tid] != 0;
        const uint32_t lo_w = diff ? (lo & ~63u) : lo;  // the mask covers whole 64-byte words
        gfs_rpc_resp rs;
        const int32_t r = rpc_call(c, GFS_OP_WRITE, fs.hfid, ((pb + tid) << c->page_shift) + lo_w, sc.stage[tid],
                                   hi - lo_w, diff ? GFS_WF_MASK : (wr >= hi - lo ? GFS_WF_FULL : 0u),
                                   diff ? (uint64_t)sc.fill[tid] : 0, nullptr, 0, &rs);
        stage_free(c, sc.stage[tid]);
        if (diff) stage_free(c, (int)sc.fill[tid]);
        if (r < 0) {
          atomicMin(&sc.err, r);
        } else {
          synced(c, f, lo, hi, wr, rs.version);
          if (diff) {
            st_rlx(&c->f_hv[f], 0);
            pristine_free(c, f);
          }
          st_rlx(&c->f_lo[f], GFS_DIRTY_NONE);
          st_rlx(&c->f_hi[f], 0);
          st_rlx(&c->f_written[f], 0);
          ctr(c, GFS_C_WRITEBACK);
          ctr(c, GFS_C_RPC_WRITE);
          ctr(c, GFS_C_BYTES_D2H, hi - lo);
        }
        a64_and_rel(&c->f_state[f], fl64(GFS_ST_EVICTING));
      }
      __syncthreads();
      if (!sc.busy) {
        ++bi;
        ns = 256;
      } else {  // some page of the batch found no staging slot: back off, redo the batch
        if (tid == 0 && timed_out(c, t0)) atomicMin(&sc.err, -ETIMEDOUT);
        __syncthreads();
        if (sc.err == -ETIMEDOUT) break;
        __nanosleep(ns);
        ns = ns < 8192 ? ns * 2 : 8192;
      }
    }
  }
  __syncthreads();
  return sc.err;
}

// gmmap: map a prefix of at most one cache page;
// returns a pointer straight into the frame, NULL at/after EOF
// or on error. *mapped_len = min(len, P - off%P, S - off). MAP_FIXED (addr) is
// ignored; prot is not enforced. Group-collective
// (G = block or warp); *err_out (optional) gets 0 or the -errno of a NULL.
template <class G>
__device__ inline void* gmmap_t(const gfs_ctx* c, void* addr, uint64_t len, int prot, int flags, int fd, uint64_t off,
                                uint64_t* mapped_len, int* err_out = nullptr) {
  using namespace detail;
  (void)addr;
  (void)flags;
  Scratch& sc = G::sc();
  const int tid = G::tid();
  const bool wmap = (prot & (int)GFS_PROT_WRITE) != 0;
  G::sync();
  if (tid == 0) {
    FileSnap s;
    sc.ptr = nullptr;
    sc.aux = 0;
    sc.ret = 0;
    if (!snap_fd_cached<G>(c, sc, fd, &s) || (s.oflags & GFS_O_GWRONCE) || (wmap && !(s.oflags & GFS_O_RDWR))) {
      sc.aux = -EBADF;  // a writable mapping needs an O_RDWR file
    } else if (off < s.size && len > 0) {
      sc.fs = s;
      sc.lc_ok = (sc.cached_fd == fd && sc.cached_blk == G::key() && sc.cached_grid == grid_id()) ? 1u : 0u;
      sc.ret = 1;
    }
  }
  G::sync();
  if (sc.ret == 1) {
    const FileSnap fs = sc.fs;
    int err = acquire_batch<G>(c, sc, fs, off >> c->page_shift, 1, false);
    if (!err && wmap) {  // writes through the pointer are untracked: keep the pristine copy, mark the range dirty
      err = ensure_pristine<G>(c, sc, fs.fdx, 1);
      if (tid == 0) {
        if (err) {
          frame_release(c, (uint32_t)sc.frame[0]);
        } else {
          const uint32_t f = (uint32_t)sc.frame[0];
          const uint64_t in = off & (c->page_size - 1);
          uint64_t m = c->page_size - in;
          if (len < m) m = len;
          if (fs.size - off < m) m = fs.size - off;
          atomicMin(&c->f_lo[f], (uint32_t)in);
          atomicMax(&c->f_hi[f], (uint32_t)(in + m));
        }
      }
    }
    if (tid == 0) {
      if (err) {
        sc.aux = err;
      } else {
        const uint64_t in = off & (c->page_size - 1);
        uint64_t m = c->page_size - in;
        if (len < m) m = len;
        if (fs.size - off < m) m = fs.size - off;
        sc.ptr = frame_ptr(c, (uint32_t)sc.frame[0]) + in;
        sc.aux = (int64_t)m;
      }
    }
    G::sync();
  }
  if constexpr (G::kBlock) {  // NEXT-2: read-ahead of a sequential mapper of a read-only file (warp 0)
    if (c->readahead && sc.ret == 1 && sc.aux > 0 && tid < 32 && !(sc.fs.oflags & GFS_O_WRITABLE) && !c->npeers &&
        ld_rlx64(&c->files[sc.fs.fdx].zc) == 0)
      ra_after<G>(c, sc, sc.fs, fd, off, (uint64_t)sc.aux);
  }
  if (mapped_len) *mapped_len = sc.aux > 0 ? (uint64_t)sc.aux : 0;
  if (err_out) *err_out = sc.aux < 0 ? (int)sc.aux : 0;
  void* const r = sc.ptr;
  if constexpr (!G::kBlock) __syncwarp();  // sc is reused by the warp's next call
  return r;
}

// gmunmap: release the page reference; the frame is found from the pointer
// (i-th pframe <-> i-th page).
template <class G>
__device__ inline int gmunmap_t(const gfs_ctx* c, void* addr, uint64_t len) {
  using namespace detail;
  (void)len;
  const uint8_t* p = (const uint8_t*)addr;
  const bool ok = p >= c->pool && p < c->pool + ((size_t)c->nframes << c->page_shift);
  if constexpr (G::kBlock) {
    Scratch& sc = G::sc();
    __syncthreads();
    if (block_tid() == 0) {
      if (ok) frame_release(c, (uint32_t)((size_t)(p - c->pool) >> c->page_shift));
      sc.ret = ok ? 0 : -EINVAL;
    }
    __syncthreads();
    return (int)sc.ret;
  } else {  // the pointer is the same in every lane: no scratch round trip
    __syncwarp();
    if (ok && G::tid() == 0) frame_release(c, (uint32_t)((size_t)(p - c->pool) >> c->page_shift));
    return ok ? 0 : -EINVAL;
  }
}

__device__ inline void* gmmap(const gfs_ctx* c, void* addr, uint64_t len, int prot, int flags, int fd, uint64_t off,
                              uint64_t* mapped_len) {
  return gmmap_t<detail::BlockGroup>(c, addr, len, prot, flags, fd, off, mapped_len);
}
__device__ inline int gmunmap(const gfs_ctx* c, void* addr, uint64_t len) {
  return gmunmap_t<detail::BlockGroup>(c, addr, len);
}
// Warp-collective gmmap / gmunmap (the paper's warp granularity):
// same semantics; a warp holds its mappings independently of the other warps.
__device__ inline void* gmmap_warp(const gfs_ctx* c, void* addr, uint64_t len, int prot, int flags, int fd,
                                   uint64_t off, uint64_t* mapped_len) {
  return gmmap_t<detail::WarpGroup>(c, addr, len, prot, flags, fd, off, mapped_len);
}
__device__ inline int gmunmap_warp(const gfs_ctx* c, void* addr, uint64_t len) {
  return gmunmap_t<detail::WarpGroup>(c, addr, len);
}

// gmsync: write back the dirty page mapped at `addr` now (Tab.1), for a
// mapping the calling block holds (gmmap with GFS_PROT_WRITE on an O_RDWR
// file). Only the bytes that differ from the page's pristine copy go to the
// host (diff-and-merge); the pristine copy then becomes the
// written-back state, so a later sync sends only later changes. The
// application coordinates gmsync with other blocks' updates (Tab.1). Returns
// 0, -EINVAL (not a mapped frame), -EBUSY (page being filled/evicted), or an
// RPC error.
__device__ inline int gmsync(const gfs_ctx* c, void* addr, uint64_t len, int flags) {
  using namespace detail;
  (void)len;
  (void)flags;
  Scratch& sc = scratch();
  const int tid = block_tid(), nthr = block_nthr();
  __syncthreads();
  if (tid == 0) {
    sc.ret = 0;
    sc.frame[0] = -1;
    const uint8_t* p = (const uint8_t*)addr;
    if (p < c->pool || p >= c->pool + ((size_t)c->nframes << c->page_shift)) {
      sc.ret = -EINVAL;
    } else {
      const uint32_t f = (uint32_t)((size_t)(p - c->pool) >> c->page_shift);
      // claim: the caller's mapping holds a reference; EVICTING keeps other
      // syncs and evictions off the page while its ranges are copied
      uint64_t v = ld_rlx64(&c->f_state[f]);
      for (;;) {
        if (((uint32_t)v & GFS_ST_REF_MASK) == 0) {
          sc.ret = -EINVAL;
          break;
        }
        if ((uint32_t)v & (GFS_ST_FILLING | GFS_ST_EVICTING | GFS_ST_ERROR)) {
          sc.ret = -EBUSY;
          break;
        }
        const uint64_t o = a64_cas(&c->f_state[f], v, v | GFS_ST_EVICTING);
        if (o == v) break;
        v = o;
      }
      if (sc.ret == 0) {
        const uint32_t lo = ld_rlx(&c->f_lo[f]), pv = ld_rlx(&c->f_pristine[f]);
        if (lo == GFS_DIRTY_NONE || pv == 0 || pv == GFS_PRISTINE_PENDING) {
          a64_and_rel(&c->f_state[f], fl64(GFS_ST_EVICTING));  // nothing written through a mapping
        } else {
          sc.frame[0] = (int)f;
          sc.lo[0] = lo;
          sc.hi[0] = ld_rlx(&c->f_hi[f]);
          sc.nbytes[0] = pv;
          sc.stage[0] = -1;
          sc.fill[0] = 0xFFFFFFFFu;
          const uint64_t t0 = now_ns();
          for (uint32_t ns = 64;;) {  // both staging slots or none
            const int a = stage_alloc(c, false);
            const int b = a >= 0 ? stage_alloc(c, false) : -1;
            if (b >= 0) {
              sc.stage[0] = a;
              sc.fill[0] = (uint32_t)b;
              break;
            }
            if (a >= 0) stage_free(c, a);
            backoff(ns);
            if (timed_out(c, t0)) {
              sc.ret = -ETIMEDOUT;
              a64_and_rel(&c->f_state[f], fl64(GFS_ST_EVICTING));
              sc.frame[0] = -1;
              break;
            }
          }
        }
      }
    }
  }
  __syncthreads();
  if (sc.frame[0] < 0) return (int)sc.ret;
  const uint32_t f = (uint32_t)sc.frame[0], lo = sc.lo[0], hi = sc.hi[0], pf = sc.nbytes[0] - 1;
  block_copy_from_frame(stage_ptr(c, sc.stage[0]) + lo, frame_ptr(c, f) + lo, hi - lo, tid, nthr);
  block_copy_from_frame(stage_ptr(c, (int)sc.fill[0]) + lo, frame_ptr(c, pf) + lo, hi - lo, tid, nthr);
  __threadfence_system();
  __syncthreads();
  if (tid == 0) {
    const uint64_t page = ld_rlx64(&c->f_tag[f]) & 0xFFFFFFFFull;
    const uint32_t fi = ld_rlx(&c->f_file[f]);
    gfs_rpc_resp rs;
    const int32_t r = rpc_call(c, GFS_OP_WRITE, ld_rlx(&c->files[fi].hfid), (page << c->page_shift) + lo,
                               sc.stage[0], hi - lo, GFS_WF_DIFF, (uint64_t)sc.fill[0], nullptr, 0, &rs);
    stage_free(c, sc.stage[0]);
    stage_free(c, (int)sc.fill[0]);
    sc.ret = r < 0 ? r : 0;
    if (r >= 0) {
      ctr(c, GFS_C_WRITEBACK);
      ctr(c, GFS_C_RPC_WRITE);
      ctr(c, GFS_C_BYTES_D2H, hi - lo);
    }
  }
  __syncthreads();
  if (sc.ret == 0)  // the written-back state is the new pristine copy
    block_copy_from_frame(frame_ptr(c, pf) + lo, frame_ptr(c, f) + lo, hi - lo, tid, nthr);
  __threadfence();
  __syncthreads();
  if (tid == 0) a64_and_rel(&c->f_state[f], fl64(GFS_ST_EVICTING));
  __syncthreads();
  return (int)sc.ret;
}

// gftruncate: reclaim the cached pages beyond the new size, clip the page the
// new EOF falls in, then ftruncate on the host (Tab.1; used by the
// mat-vec output). Pages past EOF are dropped (their dirty bytes are
// past the end of the file: discarding them is the truncate); the boundary
// page keeps only [0, size % P) — its dirty range is clipped and its tail
// zeroed — so no later write-back can grow the file again. Returns 0, or
// -EBUSY (nothing truncated on the host) if a page to drop or clip is mapped
// or in use: the caller coordinates truncation with its readers (Tab.1).
__device__ inline int gftruncate(const gfs_ctx* c, int fd, uint64_t size) {
  using namespace detail;
  Scratch& sc = scratch();
  const int tid = block_tid(), nthr = block_nthr();
  __syncthreads();
  if (tid == 0) {
    FileSnap s;
    sc.frame[0] = -1;
    if (!snap_fd(c, fd, &s) || !(s.oflags & GFS_O_WRITABLE)) {
      sc.ret = -EBADF;
    } else {
      sc.fs = s;
      sc.err = 0;
      sc.ret = 0;
    }
  }
  __syncthreads();
  if (sc.ret < 0) return (int)sc.ret;
  const FileSnap fs = sc.fs;
  const uint64_t P = c->page_size;
  const uint64_t first = (size + P - 1) >> c->page_shift;
  const uint64_t np = (fs.size + P - 1) >> c->page_shift;
  if (np > first) {
    const int r = drop_pages(c, fs, first, np, tid, nthr);
    if (r < 0) atomicMin(&sc.err, r);
  }
  const uint32_t keep = (uint32_t)(size & (P - 1));
  if (tid == 0 && keep && (size >> c->page_shift) < np) {  // the page the new EOF falls in
    const uint64_t b = size >> c->page_shift;
    uint64_t* slot = walk(c, fs.root, fs.height, b, false, nullptr);
    const uint64_t sv = slot ? ld_acq64(slot) : 0;
    if ((uint32_t)sv) {
      const uint32_t f = detail::slot_frame(sv);
      const uint64_t want = ((uint64_t)fs.uid << 32) | (uint32_t)b;
      if (ld_acq64(&c->f_tag[f]) == want) {
        if (!claim_frame(&c->f_state[f], 0u)) {
          atomicMin(&sc.err, -EBUSY);
        } else if (ld_acq64(&c->f_tag[f]) != want) {
          a64_and_rel(&c->f_state[f], fl64(GFS_ST_EVICTING));
        } else {
          const uint32_t lo = ld_rlx(&c->f_lo[f]);
          if (lo != GFS_DIRTY_NONE) {
            const uint32_t hi = ld_rlx(&c->f_hi[f]);
            if (lo >= keep) {  // every dirty byte is past the new EOF
              st_rlx(&c->f_lo[f], GFS_DIRTY_NONE);
              st_rlx(&c->f_hi[f], 0);
              st_rlx(&c->f_written[f], 0);
            } else if (hi > keep) {
              st_rlx(&c->f_hi[f], keep);
              const uint32_t wr = ld_rlx(&c->f_written[f]);
              if (wr > keep - lo) st_rlx(&c->f_written[f], keep - lo);
            }
          }
          if (ld_rlx(&c->f_valid[f]) > keep) st_rlx(&c->f_valid[f], keep);
          if (ld_rlx(&c->f_hv[f]) > keep) st_rlx(&c->f_hv[f], keep);
          sc.frame[0] = (int)f;  // the block zeroes its tail, then it is released
        }
      }
    }
  }
  __syncthreads();
  if (sc.frame[0] >= 0) {
    block_zero(frame_ptr(c, (uint32_t)sc.frame[0]) + keep, P - keep, tid, nthr);
    __threadfence();
    __syncthreads();
    if (tid == 0) a64_and_rel(&c->f_state[(uint32_t)sc.frame[0]], fl64(GFS_ST_EVICTING));
  }
  if (tid == 0 && sc.err == 0) {  // nothing cached can reach past `size` any more: truncate the host file
    const int32_t r = rpc_call(c, GFS_OP_TRUNC, fs.hfid, 0, -1, 0, 0, size, nullptr, 0, nullptr);
    if (r < 0) sc.err = r;
    else st_rlx64((uint64_t*)&c->files[fd].size, size);
  }
  __syncthreads();
  return sc.err;
}

}  // namespace gfs
