// gfs_host.cpp — host runtime of libgpufs.so: gfs_init / gfs_daemon / stats.
//
// The host side of GPUfs ("a user-level thread in the host
// application, giving it access to the application's CUDA context") and of the
// GPU-as-client RPC (§4.3). B200 redesign:
//   * the request queue is a ring of 64-byte slots in pinned, mapped host
//     memory, one queue per GPU owned by that GPU; a slot is
//     published by the GPU with st.release.sys on its seq word;
//   * W worker threads (not the paper's single event thread) each
//     claim the next ticket, spin on its slot and serve it with POSIX calls
//     only: READ preads into the pinned staging slot the GPU named, WRITE
//     pwrites from it, OPEN/CLOSE/TRUNC act on the fd table;
//   * completion is a store-release of ((ticket+1) << 32 | result) into a
//     pinned completion word that the waiting GPU thread polls with
//     ld.acquire.sys. The daemon makes NO CUDA call per request: a
//     stream-ordered DMA or stream write-value can be queued behind the very
//     kernel that waits for it when the streams share a hardware queue
//     (CUDA_DEVICE_MAX_CONNECTIONS), so the GPU pulls pages out of staging
//     itself (and pushes dirty ranges into it for write-back);
//   * a partially written dirty range is merged with the host copy by "diff
//     against zeros";
//   * close-to-open consistency uses a shared-memory version table keyed by
//     (st_dev, st_ino), bumped on every write-back (stand-in for WRAPFS,
//     P:L760-772); OPEN replies carry it so re-opens can validate.
#include <atomic>
#include <cerrno>
#include <chrono>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <deque>
#include <fcntl.h>
#include <mutex>
#include <sched.h>
#include <csetjmp>
#include <csignal>
#include <string>
#include <sys/mman.h>
#include <sys/prctl.h>
#include <sys/resource.h>
#include <sys/stat.h>
#include <thread>
#include <unistd.h>
#include <unordered_map>
#include <vector>

#include <cuda_runtime.h>

#include "gpufs.h"
#include "gfs_launch.h"

#define GFS_API extern "C" __attribute__((visibility("default")))

extern "C" int gfs_internal_init_metadata(gfs_ctx* hctx, cudaStream_t s);

namespace {

inline void cpu_relax() {
#if defined(__x86_64__)
  __builtin_ia32_pause();
#endif
}

int64_t pread_full(int fd, uint8_t* buf, uint64_t len, uint64_t off) {
  uint64_t done = 0;
  while (done < len) {
    ssize_t r = pread(fd, buf + done, len - done, (off_t)(off + done));
    if (r < 0) {
      if (errno == EINTR) continue;
      return -errno;
    }
    if (r == 0) break;
    done += (uint64_t)r;
  }
  return (int64_t)done;
}

int64_t pwrite_full(int fd, const uint8_t* buf, uint64_t len, uint64_t off) {
  uint64_t done = 0;
  while (done < len) {
    ssize_t r = pwrite(fd, buf + done, len - done, (off_t)(off + done));
    if (r < 0) {
      if (errno == EINTR) continue;
      return -errno;
    }
    done += (uint64_t)r;
  }
  return (int64_t)done;
}

// ---------------------------------------------------------------- version table
// Shared by every process on the host (one per GPU): open addressing over
// 64-bit keys mixed from (st_dev, st_ino); version bumped per write-back.
struct VEntry {
  uint64_t key;
  uint64_t version;
};
constexpr uint64_t kVEntries = 1u << 16;

struct VersionTable {
  VEntry* e = nullptr;
  bool open() {
    const char* name = getenv("GFS_VERSION_TABLE");
    std::string path = name && *name ? name : "/dev/shm/gfs_version_table_v1";
    int fd = ::open(path.c_str(), O_RDWR | O_CREAT, 0666);
    if (fd < 0) return false;
    const size_t bytes = kVEntries * sizeof(VEntry);
    struct stat st;
    if (fstat(fd, &st) != 0) { ::close(fd); return false; }
    if ((size_t)st.st_size < bytes && ftruncate(fd, (off_t)bytes) != 0) { ::close(fd); return false; }
    void* p = mmap(nullptr, bytes, PROT_READ | PROT_WRITE, MAP_SHARED, fd, 0);
    ::close(fd);
    if (p == MAP_FAILED) return false;
    e = (VEntry*)p;
    return true;
  }
  void close() {
    if (e) munmap(e, kVEntries * sizeof(VEntry));
    e = nullptr;
  }
  static uint64_t mix(uint64_t dev, uint64_t ino) {
    uint64_t z = dev * 0x9E3779B97F4A7C15ull ^ (ino + 0x632BE59BD9B4E019ull);
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
    z ^= z >> 31;
    return z | 1;
  }
  VEntry* find(uint64_t dev, uint64_t ino, bool create) {
    if (!e) return nullptr;
    const uint64_t k = mix(dev, ino);
    for (uint64_t i = 0; i < kVEntries; ++i) {
      VEntry* x = e + ((k + i) & (kVEntries - 1));
      uint64_t cur = __atomic_load_n(&x->key, __ATOMIC_ACQUIRE);
      if (cur == k) return x;
      if (cur == 0) {
        if (!create) return nullptr;
        uint64_t zero = 0;
        if (__atomic_compare_exchange_n(&x->key, &zero, k, false, __ATOMIC_ACQ_REL, __ATOMIC_ACQUIRE)) return x;
        if (zero == k) return x;
      }
    }
    return nullptr;
  }
  uint64_t get(uint64_t dev, uint64_t ino) {
    VEntry* x = find(dev, ino, false);
    return x ? __atomic_load_n(&x->version, __ATOMIC_ACQUIRE) : 0;
  }
  // Returns the new version (0 if the table is unavailable).
  uint64_t bump(uint64_t dev, uint64_t ino) {
    VEntry* x = find(dev, ino, true);
    return x ? __atomic_fetch_add(&x->version, 1, __ATOMIC_ACQ_REL) + 1 : 0;
  }
};

enum {
  HS_RPC = 0, HS_READ, HS_WRITE, HS_OPEN, HS_CLOSE, HS_TRUNC, HS_BYTES_H2D, HS_BYTES_D2H, HS_PREAD_NS,
  HS_ERRORS, HS_MERGES, HS_BUSY_NS, HS_OPEN_NS, HS_OPEN_SYS_NS, HS_OPEN_PF_NS, HS_OPEN_TAB_NS, HS_MAPPED, HS_OPEN_VT_NS, HS_N
};

}  // namespace

// One host file the GPU knows by its hfid (metadata only). Each daemon worker
// has a PRIVATE fd table (unshare(CLONE_FILES)): open()/close() in one
// process serialise on its fd-table lock, so workers sharing a table open
// files slower than one thread does. A worker re-opens a file by path the
// first time it serves it (the (dev, ino) check turns a replaced file into
// -ESTALE); `gen` invalidates cached fds when an hfid is recycled.
// Write-back of write-once files copies into a shared read-write mapping
// (see do_write): concurrent pwrite()s to one tmpfs file serialise on its
// inode lock (measured: C5 write-back stuck at ~5 GB/s with 1-16 writer
// blocks), memcpy into the page cache through a mapping does not.
constexpr uint64_t kWMapReserve = 1ull << 36;  // address space reserved per mapped file (64 GiB)
constexpr uint32_t kWMapMaxFiles = 256;

struct HostFile {
  bool live = false;
  bool map_tried = false;
  uint32_t gen = 0;
  uint32_t mode = 0;
  uint64_t dev = 0, ino = 0;
  uint64_t size = 0;        // size at (re)open
  uint8_t* map = nullptr;   // read-only shared mapping of [0, map_len), large O_RDONLY files
  uint64_t map_len = 0;
  bool wmap_tried = false;
  uint8_t* wmap = nullptr;  // read-write shared mapping (kWMapReserve bytes of address space), write-once files
  uint64_t wsize = 0;       // bytes of the file known to exist (the mapping is usable below it)
  std::string path;
};

struct WorkerFd {
  int fd;
  uint32_t gen;
};

struct Worker {
  std::thread th;
  std::vector<uint8_t> merge;
  std::unordered_map<uint32_t, WorkerFd> fds;        // hfid -> fd in this worker's table
  std::deque<uint32_t> fifo;                          // eviction order of fds
  std::unordered_map<std::string, int> dirfds;       // directory fds for openat()
  size_t cap = 1024;
  // this worker's daemon counters (HS_*): one shared array took a contended
  // atomic per counter per RPC (~9 per OPEN) and grew the per-OPEN cost with the
  // thread count; gfs_host_stats sums the workers. Own-thread relaxed adds.
  alignas(64) uint64_t hs[HS_N] = {};
  void add(int k, uint64_t v) { __atomic_fetch_add(&hs[k], v, __ATOMIC_RELAXED); }
};

// Test-and-test-and-set lock for the host file table: its critical sections
// are a few hundred nanoseconds of memory operations.
struct SpinMutex {
  std::atomic<bool> held{false};
  void lock() {
    for (;;) {
      if (!held.exchange(true, std::memory_order_acquire)) return;
      while (held.load(std::memory_order_relaxed)) cpu_relax();
    }
  }
  void unlock() { held.store(false, std::memory_order_release); }
};

struct gfs_handle {
  gfs_config cfg{};
  gfs_ctx h{};           // host copy holding device pointers
  gfs_ctx* d = nullptr;  // device copy
  bool own_pool = false;
  cudaStream_t priv = nullptr;
  gfs_rpc_req* ring_h = nullptr;
  gfs_rpc_resp* resp_h = nullptr;
  char* paths_h = nullptr;
  uint64_t* cpl_h = nullptr;
  uint8_t* staging_h = nullptr;
  std::vector<Worker> workers;
  std::atomic<uint64_t> next_ticket{0};
  std::atomic<uint64_t> frontier{0};  // one past the highest ticket whose request has arrived
  std::atomic<int64_t> last_arrival_ns{0};  // steady-clock time of the latest request
  std::atomic<bool> running{false};
  SpinMutex fd_mu;  // protects files / free_hfids (short sections: a futex sleep/wake per contended
                    // acquisition cost ~2 us per OPEN with 12 workers)
  std::vector<HostFile> files;
  uint32_t nmapped = 0;
  uint32_t nwmapped = 0;
  std::mutex grow_mu;  // file extension for mapped write-back
  std::vector<uint32_t> free_hfids;
  size_t fd_cap = 1024;  // per worker
  VersionTable vt;
  std::atomic<uint64_t> hs[HS_N];
  std::vector<gfs_peer> peers;   // views of other caches (gfs_attach_peer)
  struct ZcFile {                // gfs_register_file: a file's pages mapped for the GPU
    uint64_t dev, ino, size;
    uint8_t* map;
    uint64_t dptr;
    int fd;
    bool ro;                     // read-only mapping registered read-only
  };
  SpinMutex zc_mu;
  std::vector<ZcFile> zc;
  std::vector<void*> ipc_open;   // CUDA IPC mappings to close at shutdown
  std::atomic<uint64_t> fault_ctr{0};  // READs seen by the fault injector (gfs_config.fault)
  // Launcher argument staging (path strings for the kernels): a ring of slots
  // in pinned host + device memory of this handle's device. A slot is reused
  // only after the event recorded behind the LAST kernel that read it.
  static constexpr int kArgSlots = 64;
  char* arg_h = nullptr;
  char* arg_d = nullptr;
  cudaEvent_t arg_ev[kArgSlots] = {};
  bool arg_used[kArgSlots] = {};
  int arg_next = 0;
  std::mutex arg_mu;
};

namespace {

int cuda_err(cudaError_t e) {
  if (e == cudaSuccess) return 0;
  if (e == cudaErrorMemoryAllocation) return -ENOMEM;
  return -EIO;
}

#define CK(x)                         \
  do {                                \
    cudaError_t _e = (x);             \
    if (_e != cudaSuccess) {          \
      fprintf(stderr, "gpufs: %s failed: %s\n", #x, cudaGetErrorString(_e)); \
      rc = cuda_err(_e);              \
      goto fail;                      \
    }                                 \
  } while (0)

uint32_t alloc_hfid(gfs_handle* h, HostFile&& f, uint32_t* gen_out) {
  std::lock_guard<SpinMutex> g(h->fd_mu);
  f.live = true;
  uint32_t id;
  if (!h->free_hfids.empty()) {
    id = h->free_hfids.back();
    h->free_hfids.pop_back();
    f.gen = h->files[id].gen;
    h->files[id] = std::move(f);
  } else {
    f.gen = 0;
    h->files.push_back(std::move(f));
    id = (uint32_t)(h->files.size() - 1);
  }
  *gen_out = h->files[id].gen;
  return id;
}

// Metadata of a live hfid.
bool hfid_meta(gfs_handle* h, uint32_t id, HostFile* out) {
  std::lock_guard<SpinMutex> g(h->fd_mu);
  if (id >= h->files.size() || !h->files[id].live) return false;
  *out = h->files[id];
  return true;
}

void free_hfid(gfs_handle* h, uint32_t id) {
  uint8_t* map = nullptr;
  uint64_t map_len = 0;
  uint8_t* wmap = nullptr;
  {
    std::lock_guard<SpinMutex> g(h->fd_mu);
    if (id >= h->files.size() || !h->files[id].live) return;
    const uint32_t gen = h->files[id].gen + 1;
    map = h->files[id].map;
    map_len = h->files[id].map_len;
    wmap = h->files[id].wmap;
    if (map) --h->nmapped;
    if (wmap) --h->nwmapped;
    h->files[id] = HostFile();
    h->files[id].gen = gen;  // cached fds of the old file are now stale
    h->free_hfids.push_back(id);
  }
  // No READ or WRITE of this hfid can be in flight: the GPU closes a file only
  // after every block holding it open is done with it.
  if (map) munmap(map, map_len);
  if (wmap) munmap(wmap, kWMapReserve);
}

// ---- mapped reads --------------------------------------------------------
// READ of a large O_RDONLY file copies from a shared read-only mapping of the
// file instead of pread(): the same bytes (page cache), but one user-space
// memcpy per page instead of the kernel's per-4KiB copy loop (measured 1.4x
// per daemon thread on tmpfs). A file that shrinks under the mapping raises
// SIGBUS on access; the handler returns to the READ, which falls back to
// pread (short read, zero tail: R4).
constexpr uint64_t kMapMinBytes = 64ull << 20;
constexpr uint32_t kMapMaxFiles = 4096;
thread_local sigjmp_buf* volatile t_bus_jb = nullptr;  // volatile: the stores around memcpy must stay
struct sigaction g_old_bus;
std::once_flag g_bus_once;

void on_sigbus(int sig, siginfo_t* si, void* uc) {
  if (t_bus_jb) siglongjmp(*t_bus_jb, 1);
  if (g_old_bus.sa_flags & SA_SIGINFO) {
    if (g_old_bus.sa_sigaction) g_old_bus.sa_sigaction(sig, si, uc);
    return;
  }
  if (g_old_bus.sa_handler == SIG_DFL || g_old_bus.sa_handler == SIG_IGN) {
    signal(SIGBUS, SIG_DFL);
    raise(SIGBUS);
    return;
  }
  g_old_bus.sa_handler(sig);
}

void install_sigbus() {
  std::call_once(g_bus_once, [] {
    struct sigaction sa;
    memset(&sa, 0, sizeof(sa));
    sa.sa_sigaction = on_sigbus;
    sa.sa_flags = SA_SIGINFO | SA_NODEFER;
    sigemptyset(&sa.sa_mask);
    sigaction(SIGBUS, &sa, &g_old_bus);
  });
}

// Copy [off, off+len) of the mapping into buf; false if the access faulted.
bool map_copy(uint8_t* buf, const uint8_t* map, uint64_t off, uint64_t len) {
  sigjmp_buf jb;
  if (sigsetjmp(jb, 0) != 0) {
    t_bus_jb = nullptr;
    return false;
  }
  t_bus_jb = &jb;
  std::atomic_signal_fence(std::memory_order_seq_cst);
  memcpy(buf, map + off, len);
  std::atomic_signal_fence(std::memory_order_seq_cst);
  t_bus_jb = nullptr;
  return true;
}

// open(path) as openat(this worker's cached fd of dirname(path), basename).
int w_open_path(Worker& w, const std::string& path, int flags) {
  const size_t slash = path.rfind('/');
  if (slash == std::string::npos || slash == 0) return ::open(path.c_str(), flags, 0644);
  const std::string dir = path.substr(0, slash);
  auto it = w.dirfds.find(dir);
  int dfd;
  if (it != w.dirfds.end()) {
    dfd = it->second;
  } else {
    dfd = ::open(dir.c_str(), O_RDONLY | O_DIRECTORY | O_PATH);
    if (dfd < 0) return ::open(path.c_str(), flags, 0644);
    if (w.dirfds.size() > 4096) {  // bound the directory cache
      for (auto& kv : w.dirfds) ::close(kv.second);
      w.dirfds.clear();
    }
    w.dirfds.emplace(dir, dfd);
  }
  return ::openat(dfd, path.c_str() + slash + 1, flags, 0644);
}

void w_make_room(Worker& w) {
  while (w.fds.size() >= w.cap && !w.fifo.empty()) {
    const uint32_t id = w.fifo.front();
    w.fifo.pop_front();
    auto it = w.fds.find(id);
    if (it != w.fds.end()) {
      ::close(it->second.fd);
      w.fds.erase(it);
    }
  }
}

void w_cache(Worker& w, uint32_t id, int fd, uint32_t gen) {
  auto it = w.fds.find(id);
  if (it != w.fds.end()) {
    ::close(it->second.fd);
    it->second = WorkerFd{fd, gen};
    return;
  }
  w_make_room(w);
  w.fds.emplace(id, WorkerFd{fd, gen});
  w.fifo.push_back(id);
}

// This worker's fd for hfid (opened by path on first use). -errno on failure.
int w_fd(gfs_handle* h, Worker& w, uint32_t id) {
  auto it = w.fds.find(id);
  if (it != w.fds.end()) {  // hot path: compare the generation only (no copy of the path under the lock)
    uint32_t gen = 0;
    bool live = false;
    {
      std::lock_guard<SpinMutex> g(h->fd_mu);
      live = id < h->files.size() && h->files[id].live;
      if (live) gen = h->files[id].gen;
    }
    if (!live) return -EBADF;
    if (it->second.gen == gen) return it->second.fd;
    ::close(it->second.fd);  // the hfid was recycled for another file
    w.fds.erase(it);
  }
  HostFile m;
  if (!hfid_meta(h, id, &m)) return -EBADF;
  const int fd = w_open_path(w, m.path, (m.mode & GFS_O_WRITABLE) ? O_RDWR : O_RDONLY);
  if (fd < 0) return -errno;
  struct stat st;
  if (fstat(fd, &st) != 0 || (uint64_t)st.st_dev != m.dev || (uint64_t)st.st_ino != m.ino) {
    ::close(fd);
    return -ESTALE;
  }
  w_cache(w, id, fd, m.gen);
  return fd;
}

inline void complete(gfs_handle* h, uint32_t slot, uint64_t ticket, int32_t result) {
  __atomic_store_n(&h->cpl_h[slot], ((ticket + 1) << 32) | (uint32_t)result, __ATOMIC_RELEASE);
}

inline uint8_t* staging_slot(gfs_handle* h, uint32_t stage) {
  return h->staging_h + ((size_t)stage << h->h.page_shift);
}

int32_t do_open(gfs_handle* h, Worker& w, uint32_t slot, const gfs_rpc_req& q) {
  auto tk0 = std::chrono::steady_clock::now();
  auto lap = [&](int k) {
    const auto t = std::chrono::steady_clock::now();
    w.add(k, (uint64_t)std::chrono::duration_cast<std::chrono::nanoseconds>(t - tk0).count());
    tk0 = t;
  };
  gfs_rpc_resp* rs = h->resp_h + slot;
  std::string path(h->paths_h + (size_t)slot * GFS_MAX_PATH, q.path_len < GFS_MAX_PATH ? q.path_len : 0);
  const bool gw = (q.flags & GFS_O_WRITABLE) != 0;
  int fd = w_open_path(w, path, gw ? (O_RDWR | O_CREAT) : O_RDONLY);
  if (fd < 0) {
    rs->status = -errno;
    return rs->status;
  }
  struct stat st;
  if (fstat(fd, &st) != 0) {
    rs->status = -errno;
    ::close(fd);
    return rs->status;
  }
  lap(HS_OPEN_SYS_NS);
  // OPEN with prefetch: page 0 comes back with the reply (one RPC per small file)
  rs->pad[0] = 0;
  rs->pad[1] = 0;
  if (!gw) {  // a registered mapping of this very file (same inode and size): misses pull from it
    std::lock_guard<SpinMutex> g(h->zc_mu);
    for (const auto& z : h->zc)
      if (z.dev == (uint64_t)st.st_dev && z.ino == (uint64_t)st.st_ino && z.size == (uint64_t)st.st_size)
        rs->pad[1] = z.dptr;
  }
  if (q.stage != 0xFFFFFFFFu && !gw && q.stage < h->h.staging_slots && st.st_size > 0) {
    const uint64_t n = (uint64_t)st.st_size < h->h.page_size ? (uint64_t)st.st_size : h->h.page_size;
    uint8_t* buf = staging_slot(h, q.stage);
    const int64_t r = pread_full(fd, buf, n, 0);
    if (r >= 0) {
      if ((uint64_t)r < n) memset(buf + r, 0, n - (size_t)r);
      rs->pad[0] = n;
      w.add(HS_READ, 1);
      w.add(HS_BYTES_H2D, n);
    }
  }
  lap(HS_OPEN_PF_NS);
  uint32_t hfid;
  bool reused = false;
  if (q.arg) {  // re-open of a cached file: keep its hfid if it is the same file
    const uint32_t old = (uint32_t)(q.arg - 1);
    HostFile of;
    if (hfid_meta(h, old, &of) && of.dev == (uint64_t)st.st_dev && of.ino == (uint64_t)st.st_ino &&
        (!gw || (of.mode & GFS_O_WRITABLE))) {
      hfid = old;
      reused = true;
      // cache this fd only if it was opened as the hfid will be used: a
      // read-only re-open of a write-once hfid must not leave an O_RDONLY fd
      // where a later WRITE (pwrite) of the same hfid would find it
      if (!(of.mode & GFS_O_WRITABLE) || gw) w_cache(w, hfid, fd, of.gen);
      else ::close(fd);
    } else {
      free_hfid(h, old);
    }
  }
  if (!reused) {
    HostFile f;
    f.mode = q.flags;
    f.dev = st.st_dev;
    f.ino = st.st_ino;
    f.size = (uint64_t)st.st_size;
    f.path = std::move(path);
    uint32_t gen;
    hfid = alloc_hfid(h, std::move(f), &gen);
    w_cache(w, hfid, fd, gen);
  }
  lap(HS_OPEN_TAB_NS);
  rs->size = (int64_t)st.st_size;
  rs->version = h->vt.get(st.st_dev, st.st_ino);
  rs->ino = st.st_ino;
  rs->dev = st.st_dev;
  rs->mtime_ns = (int64_t)st.st_mtim.tv_sec * 1000000000ll + st.st_mtim.tv_nsec;
  rs->hfid = hfid;
  rs->status = 0;
  w.add(HS_OPEN, 1);
  lap(HS_OPEN_VT_NS);
  return 0;
}

// The mapping of hfid `id` (created on first use for a large O_RDONLY file).
// Returns nullptr when the file is not (or cannot be) mapped.
const uint8_t* hfid_map(gfs_handle* h, Worker& w, uint32_t id, uint64_t* map_len) {
  uint64_t size;
  uint32_t gen;
  {
    std::lock_guard<SpinMutex> g(h->fd_mu);
    if (id >= h->files.size() || !h->files[id].live) return nullptr;
    HostFile& f = h->files[id];
    if (f.map) {
      *map_len = f.map_len;
      return f.map;
    }
    if (f.map_tried || (f.mode & GFS_O_WRITABLE) || f.size < kMapMinBytes || h->nmapped >= kMapMaxFiles)
      return nullptr;
    f.map_tried = true;  // one worker maps it; the others pread meanwhile
    size = f.size;
    gen = f.gen;
  }
  const int fd = w_fd(h, w, id);
  if (fd < 0) return nullptr;
  void* p = mmap(nullptr, size, PROT_READ, MAP_SHARED, fd, 0);
  if (p == MAP_FAILED) return nullptr;
  install_sigbus();
  std::lock_guard<SpinMutex> g(h->fd_mu);
  HostFile& f = h->files[id];
  if (!f.live || f.gen != gen || f.map) {
    munmap(p, size);
    return nullptr;
  }
  f.map = (uint8_t*)p;
  f.map_len = size;
  ++h->nmapped;
  *map_len = size;
  return f.map;
}

int32_t do_read(gfs_handle* h, Worker& w, const gfs_rpc_req& q) {
  if (q.len > h->h.page_size || q.stage >= h->h.staging_slots) return -EINVAL;
  uint8_t* buf = staging_slot(h, q.stage);
  uint32_t qlen = q.len;
  if (h->cfg.fault) {  // tests: every period-th READ past a file's first page fails or comes back short
    const uint32_t kind = h->cfg.fault >> 24, period = h->cfg.fault & 0xFFFFFFu;
    if (period && q.file_off >= h->h.page_size && h->fault_ctr.fetch_add(1) % period == period - 1) {
      if (kind == GFS_FAULT_EIO) return -EIO;
      if (kind == GFS_FAULT_SHORT) qlen = q.len / 2;  // as if the file ended there: the rest reads as zeros
    }
  }
  auto t0 = std::chrono::steady_clock::now();
  uint64_t map_len = 0;
  const uint8_t* map = hfid_map(h, w, q.hfid, &map_len);
  if (!map) {  // a write-once file read back (re-opened read-only): its write mapping, below the known size
    std::lock_guard<SpinMutex> g(h->fd_mu);
    if (q.hfid < h->files.size() && h->files[q.hfid].live && h->files[q.hfid].wmap) {
      map = h->files[q.hfid].wmap;
      map_len = h->files[q.hfid].wsize;
    }
  }
  int64_t n = -1;
  if (map && q.file_off + qlen <= map_len && map_copy(buf, map, q.file_off, qlen)) {
    n = qlen;
    w.add(HS_MAPPED, 1);
  } else {
    const int fd = w_fd(h, w, q.hfid);
    if (fd < 0) return fd;
    n = pread_full(fd, buf, qlen, q.file_off);
  }
  w.add(HS_PREAD_NS, (uint64_t)std::chrono::duration_cast<std::chrono::nanoseconds>(
                            std::chrono::steady_clock::now() - t0).count());
  if (n < 0) return (int32_t)n;
  if ((uint64_t)n < q.len) memset(buf + n, 0, q.len - (size_t)n);  // host file shrank: zeros (R4)
  w.add(HS_READ, 1);
  w.add(HS_BYTES_H2D, q.len);
  return (int32_t)q.len;
}

// Copy len bytes of buf to [off, off+len) of the mapping; false if it faulted.
bool map_store(uint8_t* map, const uint8_t* buf, uint64_t off, uint64_t len) {
  sigjmp_buf jb;
  if (sigsetjmp(jb, 0) != 0) {
    t_bus_jb = nullptr;
    return false;
  }
  t_bus_jb = &jb;
  std::atomic_signal_fence(std::memory_order_seq_cst);
  memcpy(map + off, buf, len);
  std::atomic_signal_fence(std::memory_order_seq_cst);
  t_bus_jb = nullptr;
  return true;
}

// The write mapping of write-once hfid `id`, with the file grown to at least
// `end` bytes; nullptr if the file is not (or cannot be) mapped.
uint8_t* hfid_wmap(gfs_handle* h, Worker& w, uint32_t id, int fd, uint64_t end) {
  if (end > kWMapReserve) return nullptr;
  uint8_t* map;
  uint64_t wsize;
  uint32_t gen;
  bool map_it = false;
  {
    std::lock_guard<SpinMutex> g(h->fd_mu);
    if (id >= h->files.size() || !h->files[id].live) return nullptr;
    HostFile& f = h->files[id];
    map = f.wmap;
    wsize = f.wsize;
    gen = f.gen;
    if (!map) {
      if (f.wmap_tried || h->nwmapped >= kWMapMaxFiles) return nullptr;
      f.wmap_tried = true;  // one worker maps it; the others pwrite meanwhile
      map_it = true;
    }
  }
  if (map_it) {
    void* p = mmap(nullptr, kWMapReserve, PROT_READ | PROT_WRITE, MAP_SHARED | MAP_NORESERVE, fd, 0);
    if (p == MAP_FAILED) return nullptr;
    install_sigbus();
    struct stat st;
    wsize = fstat(fd, &st) == 0 ? (uint64_t)st.st_size : 0;
    std::lock_guard<SpinMutex> g(h->fd_mu);
    HostFile& f = h->files[id];
    if (!f.live || f.gen != gen || f.wmap) {
      munmap(p, kWMapReserve);
      return nullptr;
    }
    f.wmap = (uint8_t*)p;
    f.wsize = wsize;
    ++h->nwmapped;
    map = f.wmap;
  }
  if (end > wsize) {  // grow the file first: stores past EOF would fault
    std::lock_guard<std::mutex> gg(h->grow_mu);
    struct stat st;
    if (fstat(fd, &st) != 0) return nullptr;
    // fallocate only ever extends the size. ftruncate(end) here raced with a
    // concurrent pwrite() (another worker, or the fallback path) that had just
    // extended the file past `end`: it cut that write off (lost pages read
    // back as zeros, ~5% of first-iteration C5 runs)
    if ((uint64_t)st.st_size < end && fallocate(fd, 0, 0, (off_t)end) != 0) return nullptr;
    const uint64_t now = (uint64_t)st.st_size > end ? (uint64_t)st.st_size : end;
    std::lock_guard<SpinMutex> g(h->fd_mu);
    HostFile& f = h->files[id];
    if (!f.live || f.gen != gen) return nullptr;
    if (f.wsize < now) f.wsize = now;
  }
  return map;
}

int32_t do_write(gfs_handle* h, Worker& w, uint32_t slot, const gfs_rpc_req& q) {
  HostFile f;
  if (!hfid_meta(h, q.hfid, &f)) return -EBADF;
  if (!(f.mode & GFS_O_WRITABLE)) return -EBADF;  // read-only files are never written back
  const uint64_t in_page = q.file_off & (h->h.page_size - 1);
  if (in_page + q.len > h->h.page_size || q.stage >= h->h.staging_slots) return -EINVAL;
  const int fd = w_fd(h, w, q.hfid);
  if (fd < 0) return fd;
  uint8_t* buf = staging_slot(h, q.stage) + in_page;
  if (q.flags & (GFS_WF_DIFF | GFS_WF_MASK)) {
    // O_RDWR diff-and-merge: write back exactly the bytes where
    // the working copy differs from the pristine one, as runs, so bytes other
    // writers changed in the same page are never reverted
    if (!(f.mode & GFS_O_RDWR) || q.arg >= h->h.staging_slots) return -EINVAL;
    const bool bits = (q.flags & GFS_WF_MASK) != 0;  // GPU-made changed-byte mask instead of a pristine copy
    const uint8_t* pri = staging_slot(h, (uint32_t)q.arg) + (bits ? 0 : in_page);
    const uint64_t* mw = (const uint64_t*)staging_slot(h, (uint32_t)q.arg);
    auto changed = [&](uint64_t i) { return bits ? ((mw[i >> 6] >> (i & 63)) & 1) != 0 : buf[i] != pri[i]; };
    {  // the write ends at file_off + len: the file is at least that long, even if
       // its last bytes equal the pristine copy (zeros past the old EOF).
       // fallocate only ever grows the size (concurrent writers never shrink it).
      const uint64_t end = q.file_off + q.len;
      struct stat stt;
      if (fstat(fd, &stt) == 0 && (uint64_t)stt.st_size < end &&
          fallocate(fd, 0, (off_t)q.file_off, (off_t)q.len) != 0) {
        std::lock_guard<std::mutex> g(h->grow_mu);
        if (fstat(fd, &stt) == 0 && (uint64_t)stt.st_size < end && ftruncate(fd, (off_t)end) != 0) return -errno;
      }
    }
    uint8_t* wm = nullptr;
    bool wm_ok = true;
    uint64_t i = 0, runs = 0;
    while (i < q.len) {
      if (bits) {  // skip unchanged 64-byte words whole
        while (i < q.len && !(i & 63) && mw[i >> 6] == 0) i += 64;
      }
      while (i < q.len && !changed(i)) ++i;
      if (i >= q.len) break;
      uint64_t j = i;
      if (bits) {
        while (j < q.len && !(j & 63) && j + 64 <= q.len && mw[j >> 6] == ~0ull) j += 64;
      }
      while (j < q.len && changed(j)) {
        ++j;
        if (bits && !(j & 63))
          while (j + 64 <= q.len && mw[j >> 6] == ~0ull) j += 64;
      }
      if (!wm && wm_ok) {
        wm = hfid_wmap(h, w, q.hfid, fd, q.file_off + q.len);
        wm_ok = wm != nullptr;
      }
      if (!(wm && map_store(wm, buf + i, q.file_off + i, j - i))) {
        const int64_t r = pwrite_full(fd, buf + i, j - i, q.file_off + i);
        if (r < 0) return (int32_t)r;
      }
      ++runs;
      w.add(HS_BYTES_D2H, j - i);
      i = j;
    }
    h->resp_h[slot].version = h->vt.bump(f.dev, f.ino);
    w.add(HS_WRITE, 1);
    w.add(HS_MERGES, 1);
    return (int32_t)q.len;
  }
  if (!(q.flags & GFS_WF_FULL)) {
    // Not every byte of the range was written: diff against zeros.
    w.merge.assign(q.len, 0);
    int64_t r = pread_full(fd, w.merge.data(), q.len, q.file_off);
    if (r < 0) return (int32_t)r;
    for (uint32_t i = 0; i < q.len; ++i)
      if (buf[i] == 0) buf[i] = w.merge[i];
    w.add(HS_MERGES, 1);
  }
  uint8_t* wm = hfid_wmap(h, w, q.hfid, fd, q.file_off + q.len);
  if (!(wm && map_store(wm, buf, q.file_off, q.len))) {
    int64_t r = pwrite_full(fd, buf, q.len, q.file_off);
    if (r < 0) return (int32_t)r;
  } else {
    w.add(HS_MAPPED, 1);
  }
  // the version this write-back left the file at: the GPU records it as the
  // entry's synced version (peer fill); stored before completion
  h->resp_h[slot].version = h->vt.bump(f.dev, f.ino);
  w.add(HS_WRITE, 1);
  w.add(HS_BYTES_D2H, q.len);
  return (int32_t)q.len;
}

void worker_loop(gfs_handle* h, int wi) {
  Worker& w = h->workers[wi];
  w.cap = h->fd_cap;
  // A private fd table for this worker (see HostFile): its open()/close()
  // no longer contend with the other workers' on one table lock.
  unshare(CLONE_FILES);
  prctl(PR_SET_TIMERSLACK, 1000UL);  // idle sleeps end close to when asked (default slack 50 us)
  const uint32_t R = h->h.ring_slots;
  while (h->running.load(std::memory_order_acquire)) {
    const uint64_t t = h->next_ticket.fetch_add(1);
    const uint32_t slot = (uint32_t)(t % R);
    volatile gfs_rpc_req* vq = h->ring_h + slot;
    uint64_t spins = 0;
    bool stop = false;
    bool hot = false;
    while (__atomic_load_n((const uint64_t*)&vq->seq, __ATOMIC_ACQUIRE) != t + 1) {
      if (!h->running.load(std::memory_order_relaxed)) {
        stop = true;
        break;
      }
      ++spins;
      // The workers holding the next two tickets the GPU will publish poll
      // without sleeping while requests keep coming (one RPC round trip ~
      // microseconds); after 20 ms without one, and for the other workers,
      // the pause -> yield -> sleep ladder applies.
      if ((spins & 255) == 1) {
        const int64_t now = std::chrono::duration_cast<std::chrono::nanoseconds>(
                                std::chrono::steady_clock::now().time_since_epoch()).count();
        hot = t <= h->frontier.load(std::memory_order_relaxed) + 1 &&
              now - h->last_arrival_ns.load(std::memory_order_relaxed) < 20000000;
      }
      if (hot || spins < 4096) {
        cpu_relax();
      } else if (spins < 65536) {
        sched_yield();
      } else {
        usleep(50);
      }
    }
    if (stop) break;
    for (uint64_t f = h->frontier.load(std::memory_order_relaxed);
         f < t + 1 && !h->frontier.compare_exchange_weak(f, t + 1, std::memory_order_relaxed);) {
    }
    h->last_arrival_ns.store(std::chrono::duration_cast<std::chrono::nanoseconds>(
                                 std::chrono::steady_clock::now().time_since_epoch()).count(),
                             std::memory_order_relaxed);
    gfs_rpc_req q;
    q.op = vq->op;
    q.hfid = vq->hfid;
    q.file_off = vq->file_off;
    q.dev_ptr = vq->dev_ptr;
    q.len = vq->len;
    q.flags = vq->flags;
    q.arg = vq->arg;
    q.path_len = vq->path_len;
    q.stage = vq->stage;
    int32_t res;
    const auto tb = std::chrono::steady_clock::now();
    switch (q.op) {
      case GFS_OP_READ: res = do_read(h, w, q); break;
      case GFS_OP_WRITE: res = do_write(h, w, slot, q); break;
      case GFS_OP_OPEN:
        res = do_open(h, w, slot, q);
        w.add(HS_OPEN_NS, (uint64_t)std::chrono::duration_cast<std::chrono::nanoseconds>(
                                 std::chrono::steady_clock::now() - tb).count());
        break;
      case GFS_OP_CLOSE:
        free_hfid(h, q.hfid);
        w.add(HS_CLOSE, 1);
        res = 0;
        break;
      case GFS_OP_TRUNC: {
        HostFile f;
        const int fd = hfid_meta(h, q.hfid, &f) ? w_fd(h, w, q.hfid) : -EBADF;
        res = fd < 0 ? fd : (ftruncate(fd, (off_t)q.arg) == 0 ? 0 : -errno);
        if (res == 0) h->vt.bump(f.dev, f.ino);
        w.add(HS_TRUNC, 1);
        break;
      }
      case GFS_OP_NOP: res = 0; break;
      default: res = -ENOSYS;
    }
    if (res < 0) w.add(HS_ERRORS, 1);
    w.add(HS_RPC, 1);
    complete(h, slot, t, res);
    w.add(HS_BUSY_NS, (uint64_t)std::chrono::duration_cast<std::chrono::nanoseconds>(
                             std::chrono::steady_clock::now() - tb).count());
  }
  for (auto& kv : w.fds) ::close(kv.second.fd);  // this worker's private table
  for (auto& kv : w.dirfds) ::close(kv.second);
  w.fds.clear();
  w.fifo.clear();
  w.dirfds.clear();
}

void free_all(gfs_handle* h) {
  auto F = [](void* p) {
    if (p) cudaFree(p);
  };
  for (auto& z : h->zc) {
    cudaHostUnregister(z.map);
    munmap(z.map, z.size);
    ::close(z.fd);
  }
  h->zc.clear();
  for (void* p : h->ipc_open) cudaIpcCloseMemHandle(p);
  h->ipc_open.clear();
  if (h->own_pool) F(h->h.pool);
  F(h->h.f_state); F(h->h.f_tag); F(h->h.f_file); F(h->h.f_valid); F(h->h.f_lo); F(h->h.f_hi);
  F(h->h.f_written); F(h->h.f_stamp); F(h->h.f_hv); F(h->h.f_pristine); F(h->h.f_pf); F((void*)h->h.peers); F(h->h.fresh_next); F(h->h.hand); F(h->h.nodes); F(h->h.node_next);
  F(h->h.node_free); F(h->h.node_free_top); F(h->h.node_lock); F(h->h.files); F(h->h.paths); F(h->h.uid_next);
  F(h->h.ack); F(h->h.ring_tail); F(h->h.ctr); F(h->h.staging_bits); F(h->d);
  if (h->ring_h) cudaFreeHost(h->ring_h);
  if (h->resp_h) cudaFreeHost(h->resp_h);
  if (h->paths_h) cudaFreeHost(h->paths_h);
  if (h->cpl_h) cudaFreeHost(h->cpl_h);
  if (h->staging_h) cudaFreeHost(h->staging_h);
  for (int i = 0; i < gfs_handle::kArgSlots; ++i)
    if (h->arg_ev[i]) cudaEventDestroy(h->arg_ev[i]);
  F(h->arg_d);
  if (h->arg_h) cudaFreeHost(h->arg_h);
  if (h->priv) cudaStreamDestroy(h->priv);
  h->vt.close();
}

bool pow2(uint64_t x) { return x && !(x & (x - 1)); }

}  // namespace

GFS_API int gfs_config_default(gfs_config* c) {
  if (!c) return -EINVAL;
  memset(c, 0, sizeof(*c));
  c->device = 0;
  c->cache_bytes = 1ull << 30;
  c->page_size = 64u << 10;
  c->ring_slots = 4096;
  c->daemon_threads = 8;
  c->max_files = 4096;
  c->max_nodes = 0;
  c->max_batch = GFS_MAX_BATCH;
  c->flags = 0;
  c->staging_slots = 0;
  c->timeout_ms = 60000;
  return 0;
}

GFS_API int gfs_init(const gfs_config* cfg, gfs_handle** out) {
  if (!cfg || !out) return -EINVAL;
  if (!pow2(cfg->page_size) || cfg->page_size < 4096 || cfg->page_size > (16u << 20)) return -EINVAL;
  if (!pow2(cfg->ring_slots) || !pow2(cfg->max_files)) return -EINVAL;
  if (cfg->daemon_threads == 0 || cfg->daemon_threads > 256) return -EINVAL;
  const uint64_t nframes = cfg->cache_bytes / cfg->page_size;
  if (nframes == 0 || nframes >= (1ull << 31)) return -EINVAL;
  int ndev = 0;
  if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev == 0) return -ENODEV;
  if (cfg->device < 0 || cfg->device >= ndev) return -ENODEV;

  {  // the daemon keeps one host fd per cached file (a source tree is ~30k files)
    struct rlimit rl;
    if (getrlimit(RLIMIT_NOFILE, &rl) == 0 && rl.rlim_cur < rl.rlim_max) {
      rl.rlim_cur = rl.rlim_max;
      setrlimit(RLIMIT_NOFILE, &rl);
    }
  }
  gfs_handle* h = new gfs_handle();
  for (auto& x : h->hs) x = 0;
  {
    struct rlimit rl;
    const uint64_t lim = getrlimit(RLIMIT_NOFILE, &rl) == 0 ? (uint64_t)rl.rlim_cur : 1024;
    const uint64_t want = lim * 3 / 4;  // leave room for the application and other handles
    const uint64_t cap = want > 65536 ? 65536 : want;
    h->fd_cap = cap < 64 ? 64 : cap;
    const char* env = getenv("GFS_FD_CAP");  // tests: force fd-cache eviction
    if (env && atoi(env) > 0) h->fd_cap = (size_t)atoi(env);
  }
  h->cfg = *cfg;
  int rc = 0;
  gfs_ctx& c = h->h;
  const uint32_t R = cfg->ring_slots;
  const uint32_t MF = cfg->max_files;
  h->files.reserve(MF);  // host metadata grows under fd_mu: no reallocation in the OPEN path
  const uint32_t max_nodes = cfg->max_nodes ? cfg->max_nodes : (MF * 2u + 65536u);
  const size_t ctr_bytes = (size_t)GFS_C_NCOUNTERS * GFS_CTR_SHARDS * sizeof(unsigned long long);
  uint32_t slots = cfg->staging_slots;
  if (!slots) {
    const uint64_t want = (128ull << 20) / cfg->page_size;
    slots = (uint32_t)(want < 32 ? 32 : (want > 4096 ? 4096 : want));
  }
  const uint32_t words = (slots + 31) / 32;

  CK(cudaSetDevice(cfg->device));
  CK(cudaFree(0));
  CK(cudaStreamCreateWithFlags(&h->priv, cudaStreamNonBlocking));
  c.page_size = cfg->page_size;
  c.page_shift = (uint32_t)__builtin_ctz(cfg->page_size);
  c.nframes = (uint32_t)nframes;
  if (cfg->frame_pool) {
    c.pool = (uint8_t*)cfg->frame_pool;
  } else {
    CK(cudaMalloc((void**)&c.pool, nframes * cfg->page_size));
    h->own_pool = true;
  }
  CK(cudaMalloc((void**)&c.f_state, (size_t)nframes * 8));
  CK(cudaMalloc((void**)&c.f_tag, nframes * 8));
  CK(cudaMalloc((void**)&c.f_file, nframes * 4));
  CK(cudaMalloc((void**)&c.f_valid, nframes * 4));
  CK(cudaMalloc((void**)&c.f_lo, nframes * 4));
  CK(cudaMalloc((void**)&c.f_hi, nframes * 4));
  CK(cudaMalloc((void**)&c.f_written, nframes * 4));
  CK(cudaMalloc((void**)&c.f_stamp, nframes * 4));
  CK(cudaMalloc((void**)&c.f_hv, nframes * 4));
  CK(cudaMalloc((void**)&c.f_pristine, nframes * 4));
  CK(cudaMalloc((void**)&c.f_pf, nframes * 8));
  CK(cudaMalloc((void**)&c.fresh_next, 4));
  CK(cudaMalloc((void**)&c.hand, 4));
  c.max_nodes = max_nodes;
  CK(cudaMalloc((void**)&c.nodes, (size_t)max_nodes * GFS_FANOUT * 8));
  CK(cudaMalloc((void**)&c.node_next, 4));
  CK(cudaMalloc((void**)&c.node_free, (size_t)max_nodes * 4));
  CK(cudaMalloc((void**)&c.node_free_top, 4));
  CK(cudaMalloc((void**)&c.node_lock, 4));
  c.max_files = MF;
  CK(cudaMalloc((void**)&c.files, (size_t)MF * sizeof(gfs_file)));
  CK(cudaMalloc((void**)&c.paths, (size_t)MF * GFS_MAX_PATH));
  CK(cudaMalloc((void**)&c.uid_next, 4));
  c.ring_slots = R;
  CK(cudaHostAlloc((void**)&h->ring_h, (size_t)R * sizeof(gfs_rpc_req), cudaHostAllocMapped | cudaHostAllocPortable));
  CK(cudaHostAlloc((void**)&h->resp_h, (size_t)R * sizeof(gfs_rpc_resp), cudaHostAllocMapped | cudaHostAllocPortable));
  CK(cudaHostAlloc((void**)&h->paths_h, (size_t)R * GFS_MAX_PATH, cudaHostAllocMapped | cudaHostAllocPortable));
  CK(cudaHostAlloc((void**)&h->cpl_h, (size_t)R * 8, cudaHostAllocMapped | cudaHostAllocPortable));
  CK(cudaHostAlloc((void**)&h->staging_h, (size_t)slots * cfg->page_size,
                   cudaHostAllocMapped | cudaHostAllocPortable));
  memset(h->ring_h, 0, (size_t)R * sizeof(gfs_rpc_req));
  memset(h->resp_h, 0, (size_t)R * sizeof(gfs_rpc_resp));
  memset(h->cpl_h, 0, (size_t)R * 8);
  CK(cudaHostGetDevicePointer((void**)&c.ring, h->ring_h, 0));
  CK(cudaHostGetDevicePointer((void**)&c.resp, h->resp_h, 0));
  CK(cudaHostGetDevicePointer((void**)&c.ring_paths, h->paths_h, 0));
  CK(cudaHostGetDevicePointer((void**)&c.cpl, h->cpl_h, 0));
  CK(cudaHostGetDevicePointer((void**)&c.staging, h->staging_h, 0));
  c.staging_slots = slots;
  c.staging_words = words;
  CK(cudaMalloc((void**)&c.staging_bits, (size_t)words * 4));
  CK(cudaMalloc((void**)&c.ack, (size_t)R * 8));
  CK(cudaMalloc((void**)&c.ring_tail, 8));
  CK(cudaMalloc((void**)&c.ctr, ctr_bytes));
  c.flags = cfg->flags;
  c.readahead = cfg->readahead <= 8 ? cfg->readahead : 8;
  c.max_batch = cfg->max_batch >= 1 && cfg->max_batch <= GFS_MAX_BATCH ? cfg->max_batch : GFS_MAX_BATCH;
  c.timeout_ns = cfg->timeout_ms * 1000000ull;
  CK(cudaMemsetAsync(c.nodes, 0, (size_t)max_nodes * GFS_FANOUT * 8, h->priv));
  CK(cudaMemsetAsync(c.files, 0, (size_t)MF * sizeof(gfs_file), h->priv));
  CK(cudaMemsetAsync(c.paths, 0, (size_t)MF * GFS_MAX_PATH, h->priv));
  CK(cudaMemsetAsync(c.staging_bits, 0, (size_t)words * 4, h->priv));
  CK(cudaMemsetAsync(c.ack, 0, (size_t)R * 8, h->priv));
  CK(cudaMemsetAsync(c.ring_tail, 0, 8, h->priv));
  CK(cudaMemsetAsync(c.ctr, 0, ctr_bytes, h->priv));
  {
    int ir = gfs_internal_init_metadata(&c, h->priv);
    if (ir) {
      rc = ir;
      goto fail;
    }
  }
  CK(cudaMalloc((void**)&h->arg_d, (size_t)gfs_handle::kArgSlots * GFS_ARG_SLOT_BYTES));
  CK(cudaHostAlloc((void**)&h->arg_h, (size_t)gfs_handle::kArgSlots * GFS_ARG_SLOT_BYTES, cudaHostAllocPortable));
  for (int i = 0; i < gfs_handle::kArgSlots; ++i) CK(cudaEventCreateWithFlags(&h->arg_ev[i], cudaEventDisableTiming));
  CK(cudaMalloc((void**)&h->d, sizeof(gfs_ctx)));
  CK(cudaMemcpyAsync(h->d, &c, sizeof(gfs_ctx), cudaMemcpyHostToDevice, h->priv));
  CK(cudaStreamSynchronize(h->priv));
  h->workers.resize(cfg->daemon_threads);
  if (!h->vt.open()) fprintf(stderr, "gpufs: version table unavailable; close-to-open checks use size/mtime only\n");
  *out = h;
  return 0;
fail:
  free_all(h);
  delete h;
  return rc ? rc : -EIO;
}

GFS_API int gfs_daemon(gfs_handle* h, int mode) {
  if (!h) return -EINVAL;
  if (!h->running.exchange(true)) {
    for (size_t i = 0; i < h->workers.size(); ++i) h->workers[i].th = std::thread(worker_loop, h, (int)i);
  }
  if (mode == GFS_DAEMON_RUN) {
    while (h->running.load()) usleep(1000);
  }
  return 0;
}

GFS_API int gfs_daemon_stop(gfs_handle* h) {
  if (!h) return -EINVAL;
  h->running.store(false);
  for (auto& w : h->workers)
    if (w.th.joinable()) w.th.join();
  // Tickets claimed by idle workers were never posted by the GPU: restart
  // from the device's tail.
  unsigned long long tail = 0;
  cudaMemcpyAsync(&tail, h->h.ring_tail, 8, cudaMemcpyDeviceToHost, h->priv);
  cudaStreamSynchronize(h->priv);
  h->next_ticket.store(tail);
  h->frontier.store(tail);
  return 0;
}

GFS_API int gfs_shutdown(gfs_handle* h) {
  if (!h) return -EINVAL;
  gfs_daemon_stop(h);
  cudaSetDevice(h->cfg.device);
  cudaStreamSynchronize(h->priv);
  free_all(h);
  for (HostFile& f : h->files) {
    if (f.map) munmap(f.map, f.map_len);
    if (f.wmap) munmap(f.wmap, kWMapReserve);
  }
  delete h;
  return 0;
}

GFS_API const gfs_ctx* gfs_device_ctx(gfs_handle* h) { return h ? h->d : nullptr; }

// Launcher argument staging (gfs_launch.h). The strings go to a slot of this
// handle's ring (host copy, then an async copy on `s`); the caller records the
// slot's event with gfs_internal_args_done() after enqueuing the last kernel
// that reads them, and a slot is rewritten only once that event completed —
// so concurrent launches on different streams never overwrite each other's
// arguments, and the device memory belongs to the handle's own device.
extern "C" int gfs_internal_args(gfs_handle* h, cudaStream_t s, const char* const* strs, int n, char** d_out) {
  if (!h || n < 0 || n > GFS_ARG_SLOT_BYTES / GFS_MAX_PATH) return -EINVAL;
  for (int i = 0; i < n; ++i)
    if (!strs[i] || strlen(strs[i]) >= GFS_MAX_PATH) return -ENAMETOOLONG;
  std::lock_guard<std::mutex> g(h->arg_mu);
  const int k = h->arg_next;
  h->arg_next = (k + 1) % gfs_handle::kArgSlots;
  if (h->arg_used[k]) cudaEventSynchronize(h->arg_ev[k]);
  char* hp = h->arg_h + (size_t)k * GFS_ARG_SLOT_BYTES;
  for (int i = 0; i < n; ++i) memcpy(hp + (size_t)i * GFS_MAX_PATH, strs[i], strlen(strs[i]) + 1);
  char* dp = h->arg_d + (size_t)k * GFS_ARG_SLOT_BYTES;
  if (n && cudaMemcpyAsync(dp, hp, (size_t)n * GFS_MAX_PATH, cudaMemcpyHostToDevice, s) != cudaSuccess) return -EIO;
  h->arg_used[k] = false;
  *d_out = dp;
  return k;
}

extern "C" void gfs_internal_args_done(gfs_handle* h, int slot, cudaStream_t s) {
  if (!h || slot < 0 || slot >= gfs_handle::kArgSlots) return;
  std::lock_guard<std::mutex> g(h->arg_mu);
  cudaEventRecord(h->arg_ev[slot], s);
  h->arg_used[slot] = true;
}

extern "C" int gfs_internal_device(gfs_handle* h) { return h ? h->cfg.device : -1; }
extern "C" const gfs_ctx* gfs_internal_host_ctx(gfs_handle* h) { return h ? &h->h : nullptr; }

// ------------------------------------------------------------------ peer caches (NEXT-1)
namespace {
constexpr uint64_t kExportMagic = 0x3152454550534647ull;  // "GFSPEER1"
constexpr int kNExport = 7;  // pool, f_state, f_tag, f_lo, f_hv, nodes, files

int push_ctx(gfs_handle* h) {
  cudaSetDevice(h->cfg.device);
  if (cudaMemcpyAsync(h->d, &h->h, sizeof(gfs_ctx), cudaMemcpyHostToDevice, h->priv) != cudaSuccess) return -EIO;
  return cudaStreamSynchronize(h->priv) == cudaSuccess ? 0 : -EIO;
}
}  // namespace

GFS_API int gfs_export(gfs_handle* h, gfs_export_desc* out) {
  if (!h || !out) return -EINVAL;
  if (!h->own_pool) return -ENOTSUP;  // IPC needs allocation bases; a caller-owned pool may be a sub-allocation
  cudaSetDevice(h->cfg.device);
  memset(out, 0, sizeof(*out));
  out->magic = kExportMagic;
  out->pid = (int32_t)getpid();
  out->device = h->cfg.device;
  out->page_shift = h->h.page_shift;
  out->nframes = h->h.nframes;
  out->max_nodes = h->h.max_nodes;
  out->max_files = h->h.max_files;
  const void* ptrs[kNExport] = {h->h.pool, h->h.f_state, h->h.f_tag, h->h.f_lo, h->h.f_hv, h->h.nodes, h->h.files};
  for (int i = 0; i < kNExport; ++i) {
    out->ptr[i] = (uint64_t)(uintptr_t)ptrs[i];
    cudaIpcMemHandle_t m;
    if (cudaIpcGetMemHandle(&m, (void*)ptrs[i]) != cudaSuccess) return -EIO;
    static_assert(sizeof(m) == sizeof(out->ipc[0]), "IPC handle size");
    memcpy(out->ipc[i], &m, sizeof(m));
  }
  if (!(h->h.flags & GFS_F_EXPORTED)) {  // fills publish at system scope from now on
    h->h.flags |= GFS_F_EXPORTED;
    const int r = push_ctx(h);
    if (r) return r;
  }
  return 0;
}

GFS_API int gfs_attach_peer(gfs_handle* h, const gfs_export_desc* d) {
  if (!h || !d || d->magic != kExportMagic) return -EINVAL;
  if (d->page_shift != h->h.page_shift) return -EINVAL;  // frames are copied whole-page
  if (d->nframes >= (1u << 27) || !d->max_files || (d->max_files & (d->max_files - 1))) return -EINVAL;
  if (h->peers.size() >= GFS_MAX_PEERS) return -ENOSPC;
  const bool local = d->pid == (int32_t)getpid();
  if (local && d->ptr[0] == (uint64_t)(uintptr_t)h->h.pool) return -EINVAL;  // itself
  cudaSetDevice(h->cfg.device);
  void* p[kNExport] = {};
  if (local) {
    if (d->device != h->cfg.device) {
      const cudaError_t e = cudaDeviceEnablePeerAccess(d->device, 0);
      if (e != cudaSuccess && e != cudaErrorPeerAccessAlreadyEnabled) return -EIO;
      cudaGetLastError();
    }
    for (int i = 0; i < kNExport; ++i) p[i] = (void*)(uintptr_t)d->ptr[i];
  } else {
    for (int i = 0; i < kNExport; ++i) {
      cudaIpcMemHandle_t m;
      memcpy(&m, d->ipc[i], sizeof(m));
      if (cudaIpcOpenMemHandle(&p[i], m, cudaIpcMemLazyEnablePeerAccess) != cudaSuccess) {
        fprintf(stderr, "gpufs: cudaIpcOpenMemHandle failed: %s\n", cudaGetErrorString(cudaGetLastError()));
        for (int j = 0; j < i; ++j) cudaIpcCloseMemHandle(p[j]);
        return -EIO;
      }
    }
    for (int i = 0; i < kNExport; ++i) h->ipc_open.push_back(p[i]);
  }
  gfs_peer v{};
  v.pool = (uint8_t*)p[0];
  v.f_state = (uint64_t*)p[1];
  v.f_tag = (uint64_t*)p[2];
  v.f_lo = (uint32_t*)p[3];
  v.f_hv = (uint32_t*)p[4];
  v.nodes = (uint64_t*)p[5];
  v.files = (gfs_file*)p[6];
  v.nframes = d->nframes;
  v.max_nodes = d->max_nodes;
  v.max_files = d->max_files;
  v.page_shift = d->page_shift;
  h->peers.push_back(v);
  if (!h->h.peers && cudaMalloc((void**)&h->h.peers, GFS_MAX_PEERS * sizeof(gfs_peer)) != cudaSuccess) return -ENOMEM;
  if (cudaMemcpy((void*)h->h.peers, h->peers.data(), h->peers.size() * sizeof(gfs_peer), cudaMemcpyHostToDevice) !=
      cudaSuccess)
    return -EIO;
  h->h.npeers = (uint32_t)h->peers.size();
  const int r = push_ctx(h);
  return r ? r : (int)h->peers.size() - 1;
}

GFS_API int gfs_register_file(gfs_handle* h, const char* path) {
  if (!h || !path) return -EINVAL;
  cudaSetDevice(h->cfg.device);
  // First a read-only registration of a read-only mapping (the GPU only pulls
  // from it; an input the caller cannot write can be registered, and no
  // device store can reach the file). Drivers that refuse to register a
  // PROT_READ mapping get the read-write mapping instead (measured in round 1
  // on this image: cudaHostRegister of a PROT_READ mapping -> invalid argument).
  for (int attempt = 0; attempt < 2; ++attempt) {
    const bool ro = attempt == 0;
    const int fd = ::open(path, ro ? O_RDONLY : O_RDWR);
    if (fd < 0) {
      if (ro) continue;
      return -errno;
    }
    struct stat st;
    if (fstat(fd, &st) != 0) {
      const int e = -errno;
      ::close(fd);
      return e;
    }
    if (st.st_size <= 0) {
      ::close(fd);
      return -EINVAL;
    }
    const uint64_t size = (uint64_t)st.st_size;
    void* m = mmap(nullptr, size, ro ? PROT_READ : (PROT_READ | PROT_WRITE), MAP_SHARED, fd, 0);
    if (m == MAP_FAILED) {
      const int e = -errno;
      ::close(fd);
      return e;
    }
    void* d = nullptr;
    const unsigned flags = cudaHostRegisterMapped | (ro ? cudaHostRegisterReadOnly : 0u);
    if (cudaHostRegister(m, size, flags) != cudaSuccess || cudaHostGetDevicePointer(&d, m, 0) != cudaSuccess) {
      const cudaError_t e = cudaGetLastError();  // clears the error for the next attempt
      munmap(m, size);
      ::close(fd);
      if (ro) continue;
      fprintf(stderr, "gpufs: cudaHostRegister(%s): %s\n", path, cudaGetErrorString(e));
      return -EIO;
    }
    std::lock_guard<SpinMutex> g(h->zc_mu);
    h->zc.push_back({(uint64_t)st.st_dev, (uint64_t)st.st_ino, size, (uint8_t*)m, (uint64_t)(uintptr_t)d, fd, ro});
    return ro ? 1 : 0;
  }
  return -EIO;
}

GFS_API int gfs_stats(gfs_handle* h, uint64_t* out, int n, int reset) {
  if (!h || !out) return -EINVAL;
  std::vector<unsigned long long> buf((size_t)GFS_C_NCOUNTERS * GFS_CTR_SHARDS);
  cudaSetDevice(h->cfg.device);
  if (cudaMemcpyAsync(buf.data(), h->h.ctr, buf.size() * 8, cudaMemcpyDeviceToHost, h->priv) != cudaSuccess)
    return -EIO;
  if (cudaStreamSynchronize(h->priv) != cudaSuccess) return -EIO;
  for (int i = 0; i < n && i < GFS_C_NCOUNTERS; ++i) {
    uint64_t s = 0;
    for (int k = 0; k < GFS_CTR_SHARDS; ++k) s += buf[(size_t)i * GFS_CTR_SHARDS + k];
    out[i] = s;
  }
  if (reset) {
    cudaMemsetAsync(h->h.ctr, 0, buf.size() * 8, h->priv);
    cudaStreamSynchronize(h->priv);
  }
  return GFS_C_NCOUNTERS;
}

GFS_API int gfs_host_stats(gfs_handle* h, uint64_t* out, int n) {
  if (!h || !out) return -EINVAL;
  for (int i = 0; i < n && i < HS_N; ++i) {
    uint64_t v = h->hs[i].load();
    for (const Worker& w : h->workers) v += __atomic_load_n(&w.hs[i], __ATOMIC_RELAXED);
    out[i] = v;
  }
  return HS_N;
}

GFS_API int gfs_info(gfs_handle* h, uint64_t* out, int n) {
  if (!h || !out) return -EINVAL;
  unsigned long long tail = 0;
  cudaMemcpyAsync(&tail, h->h.ring_tail, 8, cudaMemcpyDeviceToHost, h->priv);
  cudaStreamSynchronize(h->priv);
  uint64_t v[9] = {h->h.page_size, h->h.nframes, h->h.max_files, h->h.max_nodes, h->h.ring_slots,
                   h->workers.size(), h->h.staging_slots, h->next_ticket.load(), tail};
  for (int i = 0; i < n && i < 9; ++i) out[i] = v[i];
  return 9;
}
