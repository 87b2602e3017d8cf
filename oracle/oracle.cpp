// oracle/oracle.cpp — the CPU oracle for the GPUfs buffer-cache read path.
//
// TEST INFRASTRUCTURE ONLY. Only tests/, __graft_entry__.smoke() and bench.py's
// cpu_baseline / --impl reference legs may load this library. The product path
// (paper_conf_asplos_silbersteinfkw13_b200/) never links, imports or calls it,
// and shares no code, header, table or helper with it.
//
// Plain, slow, obviously-correct C++17 over POSIX open/pread/pwrite/fstat.
// Every function cites the PAPER.md passage (P:L<line>, /root/reference/PAPER.md)
// whose definition it writes out. Where the paper is silent the reading taken is
// the one listed in DESIGN.md §"Readings" (mirrors SURVEY.md §8(c)).
//
// Pinned by tests/test_oracle_*.py against: raw pread (library special case),
// brute-force grep -w on tiny corpora, GNU grep -owF, closed-form splitmix
// content, integer-valued mat-vec (exact), and the page-cache counter
// invariants of SURVEY §8(c) O1. Functions with no such pin say so below.

#include <algorithm>
#include <cerrno>
#include <climits>
#include <cstdint>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <fcntl.h>
#include <list>
#include <map>
#include <mutex>
#include <string>
#include <sys/stat.h>
#include <thread>
#include <unistd.h>
#include <unordered_map>
#include <vector>

#define ORC_API extern "C" __attribute__((visibility("default")))

// ---------------------------------------------------------------------------
// POSIX helpers: loop on short reads/writes and EINTR.
// ---------------------------------------------------------------------------
static int64_t pread_full(int fd, uint8_t* buf, uint64_t len, uint64_t off) {
  uint64_t done = 0;
  while (done < len) {
    ssize_t r = pread(fd, buf + done, len - done, (off_t)(off + done));
    if (r < 0) {
      if (errno == EINTR) continue;
      return -errno;
    }
    if (r == 0) break;  // host file is shorter than requested
    done += (uint64_t)r;
  }
  return (int64_t)done;
}

static int64_t pwrite_full(int fd, const uint8_t* buf, uint64_t len, uint64_t off) {
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

// ---------------------------------------------------------------------------
// O1 — gread as a plain definition (§3.2: gread corresponds to
// POSIX pread with an explicit offset; Tab.1: the file size is the size
// at the first gopen). Result = the bytes pread returns for
// [off, off + min(len, S - off)), 0 bytes when off >= S. If the host file is
// now shorter than the snapshot S the missing tail reads as zeros (reading R4
// in DESIGN.md).
// ---------------------------------------------------------------------------
ORC_API int64_t orc_pread(const char* path, uint64_t snap_size, uint64_t off, uint64_t len,
                          uint8_t* out) {
  int fd = open(path, O_RDONLY);
  if (fd < 0) return -errno;
  uint64_t n = off >= snap_size ? 0 : std::min(len, snap_size - off);
  int64_t r = n ? pread_full(fd, out, n, off) : 0;
  close(fd);
  if (r < 0) return r;
  if ((uint64_t)r < n) memset(out + r, 0, n - (uint64_t)r);
  return (int64_t)n;
}

ORC_API int64_t orc_file_size(const char* path) {
  struct stat st;
  if (stat(path, &st) != 0) return -errno;
  return (int64_t)st.st_size;
}

// ---------------------------------------------------------------------------
// The C2 consumer result: a position-weighted checksum of the bytes read.
// sum over 8-byte words j overlapping [off, off+len) of  w_j * (2j + 1)  mod 2^64,
// where w_j is the little-endian value of file bytes [8j, 8j+8) with bytes
// outside [off, off+len) (and beyond EOF) taken as zero. (R9; the
// paper's K1 does not touch the data, P:L827-828 — the checksum is ours, so the
// sweep is checked end to end.)
// ---------------------------------------------------------------------------
ORC_API int64_t orc_checksum(const char* path, uint64_t off, uint64_t len, uint64_t* out_sum) {
  int fd = open(path, O_RDONLY);
  if (fd < 0) return -errno;
  const uint64_t chunk = 1ull << 22;
  std::vector<uint8_t> buf(chunk + 16);
  uint64_t sum = 0;
  uint64_t pos = off, end = off + len;
  while (pos < end) {
    uint64_t n = std::min(chunk, end - pos);
    int64_t r = pread_full(fd, buf.data(), n, pos);
    if (r < 0) { close(fd); return r; }
    if ((uint64_t)r < n) memset(buf.data() + r, 0, n - (uint64_t)r);
    for (uint64_t i = 0; i < n; ++i) {
      uint64_t o = pos + i;
      uint64_t j = o >> 3;
      uint64_t b = (uint64_t)buf[i] << (8 * (o & 7));
      sum += b * (2 * j + 1);
    }
    pos += n;
  }
  close(fd);
  *out_sum = sum;
  return 0;
}

// The same definition over a large range with T threads: the sum is over
// bytes (each byte b at offset o adds (b << 8(o mod 8)) * (2(o div 8) + 1)),
// so [off, off+len) is cut into T contiguous pieces, each summed by
// orc_checksum above, and the pieces' sums are added mod 2^64. Used to check
// the C2 sweep at its full size (8 GiB) in bench.py.
ORC_API int64_t orc_checksum_mt(const char* path, uint64_t off, uint64_t len, int nthreads, uint64_t* out_sum) {
  if (nthreads < 1) nthreads = 1;
  std::vector<uint64_t> part(nthreads, 0);
  std::vector<int64_t> rc(nthreads, 0);
  std::vector<std::thread> th;
  const uint64_t per = (len + nthreads - 1) / nthreads;
  for (int t = 0; t < nthreads; ++t)
    th.emplace_back([&, t]() {
      const uint64_t a = std::min(len, per * (uint64_t)t), b = std::min(len, a + per);
      if (b > a) rc[t] = orc_checksum(path, off + a, b - a, &part[t]);
    });
  for (auto& x : th) x.join();
  uint64_t sum = 0;
  for (int t = 0; t < nthreads; ++t) {
    if (rc[t] < 0) return rc[t];
    sum += part[t];
  }
  *out_sum = sum;
  return 0;
}

// K4: the consumer adds the checksum of every chunk it reads;
// the expected total is the sum over calls i of checksum(offs[i], len) — each
// call's bytes read with pread, calls split over T threads.
ORC_API int64_t orc_checksum_calls(const char* path, const uint64_t* offs, uint64_t ncalls, uint64_t len,
                                   int nthreads, uint64_t* out_sum) {
  if (nthreads < 1) nthreads = 1;
  std::vector<uint64_t> part(nthreads, 0);
  std::vector<int64_t> rc(nthreads, 0);
  std::vector<std::thread> th;
  for (int t = 0; t < nthreads; ++t)
    th.emplace_back([&, t]() {
      int fd = open(path, O_RDONLY);
      if (fd < 0) {
        rc[t] = -errno;
        return;
      }
      std::vector<uint8_t> buf(len + 1);
      uint64_t sum = 0;
      for (uint64_t i = (uint64_t)t; i < ncalls; i += (uint64_t)nthreads) {
        const int64_t r = pread_full(fd, buf.data(), len, offs[i]);
        if (r < 0) {
          rc[t] = r;
          break;
        }
        if ((uint64_t)r < len) memset(buf.data() + r, 0, len - (uint64_t)r);
        for (uint64_t k = 0; k < len; ++k) {
          const uint64_t o = offs[i] + k;
          sum += ((uint64_t)buf[k] << (8 * (o & 7))) * (2 * (o >> 3) + 1);
        }
      }
      close(fd);
      part[t] = sum;
    });
  for (auto& x : th) x.join();
  uint64_t sum = 0;
  for (int t = 0; t < nthreads; ++t) {
    if (rc[t] < 0) return rc[t];
    sum += part[t];
  }
  *out_sum = sum;
  return 0;
}

// ---------------------------------------------------------------------------
// Page-cache model (O1/O2): the simple buffer cache of P:L587-622 §4.2 with
// per-file page lookup, an LRU of capacity C pages (the north star's
// "LRU/refcount" policy; any victim is correct, only counters depend on it),
// O_GWRONCE pages that are never fetched and whose pristine copy is zeros
// (§3.1), gclose without write-back,
// gfsync writing back dirty pages (Tab.1), and lazy
// invalidation on re-open (§4.4) keyed by a per-path version that
// every write-back bumps (the user-space stand-in for WRAPFS, R7),
// and O_RDWR write sharing: pages are fetched, a pristine copy is
// preserved before the first local write (R21), and write-back sends
// only the bytes where the working copy differs from the pristine one.
// ---------------------------------------------------------------------------
namespace {

std::mutex g_ver_mu;
std::map<std::string, uint64_t> g_versions;  // process-wide "version table"

uint64_t version_of(const std::string& p) {
  std::lock_guard<std::mutex> g(g_ver_mu);
  return g_versions[p];
}
void version_bump(const std::string& p) {
  std::lock_guard<std::mutex> g(g_ver_mu);
  g_versions[p] += 1;
}

struct OFile {
  std::string path;
  int hfd = -1;
  uint64_t size = 0;       // snapshot at first gopen, max written end if writable
  bool gwronce = false;
  bool rdwr = false;
  uint64_t version = 0;
  uint64_t uid = 0;
  int refs = 0;
};

struct OPage {
  std::vector<uint8_t> data;  // P bytes
  bool dirty = false;
  uint64_t lo = 0, hi = 0;    // dirty byte range within the page
  uint64_t written = 0;       // bytes written into the page by gwrite
  std::vector<uint8_t> pristine;  // O_RDWR: copy taken before the first local write (empty: none)
  int file = -1;
};

typedef std::pair<uint64_t, uint64_t> PKey;  // (uid, page index)

struct OCache {
  uint64_t P = 0, cap = 0;
  uint64_t next_uid = 1;
  std::vector<OFile> files;
  std::map<PKey, OPage> pages;
  std::list<PKey> lru;  // front = most recently used
  std::map<PKey, std::list<PKey>::iterator> lru_pos;
  uint64_t hits = 0, misses = 0, evictions = 0, writebacks = 0;
};

int64_t writeback(OCache* c, OPage& pg, const PKey& k) {
  if (!pg.dirty) return 0;
  OFile& f = c->files[pg.file];
  uint64_t base = k.second * c->P;
  uint64_t n = pg.hi - pg.lo;
  if (!pg.pristine.empty()) {
    // O_RDWR: "diff" the working and pristine copies and write
    // only the bytes that differ; the file is extended to the write's end.
    struct stat st;
    if (fstat(f.hfd, &st) != 0) return -errno;
    if ((uint64_t)st.st_size < base + pg.hi && ftruncate(f.hfd, (off_t)(base + pg.hi)) != 0) return -errno;
    for (uint64_t i = pg.lo; i < pg.hi; ++i) {
      if (pg.data[i] == pg.pristine[i]) continue;
      int64_t r = pwrite_full(f.hfd, &pg.data[i], 1, base + i);
      if (r < 0) return r;
    }
    pg.pristine.clear();
    pg.dirty = false;
    pg.lo = pg.hi = pg.written = 0;
    c->writebacks++;
    version_bump(f.path);
    f.version = version_of(f.path);
    return 0;
  }
  std::vector<uint8_t> out(pg.data.begin() + pg.lo, pg.data.begin() + pg.hi);
  if (pg.written < n) {
    // Not every byte of [lo,hi) was written: "diff against zeros"
    // — a zero byte in the working copy keeps the host byte.
    std::vector<uint8_t> host(n, 0);
    int64_t r = pread_full(f.hfd, host.data(), n, base + pg.lo);
    if (r < 0) return r;
    for (uint64_t i = 0; i < n; ++i)
      if (out[i] == 0) out[i] = host[i];
  }
  int64_t r = pwrite_full(f.hfd, out.data(), n, base + pg.lo);
  if (r < 0) return r;
  pg.dirty = false;
  pg.lo = pg.hi = pg.written = 0;
  c->writebacks++;
  version_bump(f.path);
  f.version = version_of(f.path);
  return 0;
}

void touch(OCache* c, const PKey& k) {
  auto it = c->lru_pos.find(k);
  if (it != c->lru_pos.end()) c->lru.erase(it->second);
  c->lru.push_front(k);
  c->lru_pos[k] = c->lru.begin();
}

void drop_page(OCache* c, const PKey& k) {
  auto it = c->lru_pos.find(k);
  if (it != c->lru_pos.end()) {
    c->lru.erase(it->second);
    c->lru_pos.erase(it);
  }
  c->pages.erase(k);
}

int64_t make_room(OCache* c) {
  while (c->pages.size() >= c->cap && !c->lru.empty()) {
    PKey victim = c->lru.back();
    OPage& pg = c->pages[victim];
    int64_t r = writeback(c, pg, victim);
    if (r < 0) return r;
    drop_page(c, victim);
    c->evictions++;
  }
  return 0;
}

// Drop every cached page of one file incarnation (after writing back dirty ones).
int64_t drop_file_pages(OCache* c, uint64_t uid) {
  std::vector<PKey> ks;
  for (auto& kv : c->pages)
    if (kv.first.first == uid) ks.push_back(kv.first);
  for (auto& k : ks) {
    int64_t r = writeback(c, c->pages[k], k);
    if (r < 0) return r;
    drop_page(c, k);
  }
  return 0;
}

// Find-or-load the page (uid, p) of file fidx. Returns nullptr on error (*err set).
OPage* get_page(OCache* c, int fidx, uint64_t p, int64_t* err) {
  OFile& f = c->files[fidx];
  PKey k(f.uid, p);
  auto it = c->pages.find(k);
  if (it != c->pages.end()) {
    c->hits++;
    touch(c, k);
    return &it->second;
  }
  c->misses++;
  int64_t r = make_room(c);
  if (r < 0) { *err = r; return nullptr; }
  OPage pg;
  pg.data.assign(c->P, 0);
  pg.file = fidx;
  if (!f.gwronce) {
    // Miss: fetch min(P, S - pP) bytes of the page from the host.
    uint64_t base = p * c->P;
    uint64_t n = base >= f.size ? 0 : std::min<uint64_t>(c->P, f.size - base);
    if (n) {
      int64_t rr = pread_full(f.hfd, pg.data.data(), n, base);
      if (rr < 0) { *err = rr; return nullptr; }
    }
  }
  // O_GWRONCE: never fetched; pristine copy is zeros.
  auto ins = c->pages.emplace(k, std::move(pg));
  touch(c, k);
  return &ins.first->second;
}

}  // namespace

ORC_API void* orc_cache_new(uint64_t page_size, uint64_t capacity_pages) {
  if (page_size == 0 || capacity_pages == 0) return nullptr;
  OCache* c = new OCache();
  c->P = page_size;
  c->cap = capacity_pages;
  return c;
}

ORC_API void orc_cache_free(void* h) {
  OCache* c = (OCache*)h;
  if (!c) return;
  for (auto& f : c->files)
    if (f.hfd >= 0) close(f.hfd);
  delete c;
}

// flags: 0 = O_RDONLY, 1 = O_GWRONCE, 2 = O_RDWR.
ORC_API int orc_cache_open(void* h, const char* path, int flags) {
  OCache* c = (OCache*)h;
  if (flags < 0 || flags > 2) return -EINVAL;
  const bool rw = flags == 2;
  bool gw = flags == 1;
  std::string p(path);
  for (size_t i = 0; i < c->files.size(); ++i) {
    OFile& f = c->files[i];
    if (f.path != p) continue;
    if (f.refs > 0) {
      // Already open on this GPU: the fd is shared.
      if (f.gwronce != gw || f.rdwr != rw) return -EBUSY;  // one mode at a time
      f.refs++;
      return (int)i;
    }
    // Closed-file cache: re-open validates.
    struct stat st;
    if (stat(path, &st) != 0) return -errno;
    bool stale = gw || rw || f.gwronce || f.rdwr || version_of(p) != f.version || (uint64_t)st.st_size != f.size;
    if (stale) {
      int64_t r = drop_file_pages(c, f.uid);
      if (r < 0) return (int)r;
      if (f.hfd >= 0) close(f.hfd);
      f.hfd = (gw || rw) ? open(path, O_RDWR | O_CREAT, 0644) : open(path, O_RDONLY);
      if (f.hfd < 0) return -errno;
      if (fstat(f.hfd, &st) != 0) return -errno;
      f.uid = c->next_uid++;
      f.size = (uint64_t)st.st_size;
      f.gwronce = gw;
      f.rdwr = rw;
      f.version = version_of(p);
    }
    f.refs = 1;
    return (int)i;
  }
  OFile f;
  f.path = p;
  f.hfd = (gw || rw) ? open(path, O_RDWR | O_CREAT, 0644) : open(path, O_RDONLY);
  if (f.hfd < 0) return -errno;
  struct stat st;
  if (fstat(f.hfd, &st) != 0) return -errno;
  f.size = (uint64_t)st.st_size;
  f.gwronce = gw;
  f.rdwr = rw;
  f.version = version_of(p);
  f.uid = c->next_uid++;
  f.refs = 1;
  c->files.push_back(f);
  return (int)(c->files.size() - 1);
}

// gclose: refcount-- ; never writes back.
ORC_API int orc_cache_close(void* h, int fd) {
  OCache* c = (OCache*)h;
  if (fd < 0 || (size_t)fd >= c->files.size() || c->files[fd].refs <= 0) return -EBADF;
  c->files[fd].refs--;
  return 0;
}

ORC_API int64_t orc_cache_size(void* h, int fd) {
  OCache* c = (OCache*)h;
  if (fd < 0 || (size_t)fd >= c->files.size() || c->files[fd].refs <= 0) return -EBADF;
  return (int64_t)c->files[fd].size;
}

// gread through the model: per page in the span, look it up (loading on a
// miss, evicting LRU), then copy the slice (Fig. 3 / P:L570-576).
ORC_API int64_t orc_cache_read(void* h, int fd, uint64_t off, uint64_t len, uint8_t* out) {
  OCache* c = (OCache*)h;
  if (fd < 0 || (size_t)fd >= c->files.size() || c->files[fd].refs <= 0) return -EBADF;
  OFile& f = c->files[fd];
  if (f.gwronce) return -EBADF;  // write-only file
  uint64_t n = off >= f.size ? 0 : std::min(len, f.size - off);
  uint64_t done = 0;
  while (done < n) {
    uint64_t o = off + done;
    uint64_t p = o / c->P, in = o % c->P;
    uint64_t take = std::min(c->P - in, n - done);
    int64_t err = 0;
    OPage* pg = get_page(c, fd, p, &err);
    if (!pg) return err;
    memcpy(out + done, pg->data.data() + in, take);
    done += take;
  }
  return (int64_t)n;
}

// gmmap through the model: the mapped prefix is min(len, P - off%P, S - off)
// (at most one page P:L990-991); its bytes are copied to out.
ORC_API int64_t orc_cache_mmap_copy(void* h, int fd, uint64_t off, uint64_t len, uint8_t* out) {
  OCache* c = (OCache*)h;
  if (fd < 0 || (size_t)fd >= c->files.size() || c->files[fd].refs <= 0) return -EBADF;
  OFile& f = c->files[fd];
  if (off >= f.size) return 0;
  uint64_t n = std::min(std::min(len, c->P - off % c->P), f.size - off);
  return orc_cache_read(h, fd, off, n, out);
}

// gwrite on an O_GWRONCE file: pages are zero-initialised, never fetched;
// on an O_RDWR file: pages are fetched and keep a pristine copy from before
// the first local write. The dirty range and written-byte count are tracked;
// size grows.
ORC_API int64_t orc_cache_write(void* h, int fd, uint64_t off, uint64_t len, const uint8_t* in) {
  OCache* c = (OCache*)h;
  if (fd < 0 || (size_t)fd >= c->files.size() || c->files[fd].refs <= 0) return -EBADF;
  OFile& f = c->files[fd];
  if (!f.gwronce && !f.rdwr) return -EBADF;
  uint64_t done = 0;
  while (done < len) {
    uint64_t o = off + done;
    uint64_t p = o / c->P, in_off = o % c->P;
    uint64_t take = std::min(c->P - in_off, len - done);
    int64_t err = 0;
    OPage* pg = get_page(c, fd, p, &err);
    if (!pg) return err;
    if (f.rdwr && pg->pristine.empty()) pg->pristine = pg->data;
    memcpy(pg->data.data() + in_off, in + done, take);
    if (!pg->dirty) {
      pg->dirty = true;
      pg->lo = in_off;
      pg->hi = in_off + take;
    } else {
      pg->lo = std::min<uint64_t>(pg->lo, in_off);
      pg->hi = std::max<uint64_t>(pg->hi, in_off + take);
    }
    pg->written += take;
    done += take;
  }
  f.size = std::max(f.size, off + len);
  return (int64_t)len;
}

// A writable gmmap of an O_RDWR file, stores through it, and (do_msync) gmsync
// (Tab.1, R22/R23): the mapped prefix m = min(len, P - off%P,
// S - off) is written; the page keeps its pristine copy and the range is
// dirty; gmsync writes the page's diff back now and makes the written-back
// state the new pristine copy (the page stays dirty: the mapping may be
// written again). Returns m.
ORC_API int64_t orc_cache_mmap_write(void* h, int fd, uint64_t off, uint64_t len, const uint8_t* in,
                                     int do_msync) {
  OCache* c = (OCache*)h;
  if (fd < 0 || (size_t)fd >= c->files.size() || c->files[fd].refs <= 0) return -EBADF;
  OFile& f = c->files[fd];
  if (!f.rdwr) return -EBADF;
  if (off >= f.size || len == 0) return 0;
  const uint64_t p = off / c->P, in_off = off % c->P;
  const uint64_t m = std::min(std::min(len, c->P - in_off), f.size - off);
  int64_t err = 0;
  OPage* pg = get_page(c, fd, p, &err);
  if (!pg) return err;
  if (pg->pristine.empty()) pg->pristine = pg->data;
  memcpy(pg->data.data() + in_off, in, m);
  if (!pg->dirty) {
    pg->dirty = true;
    pg->lo = in_off;
    pg->hi = in_off + m;
  } else {
    pg->lo = std::min<uint64_t>(pg->lo, in_off);
    pg->hi = std::max<uint64_t>(pg->hi, in_off + m);
  }
  if (do_msync) {
    const PKey k(f.uid, p);
    const uint64_t lo = pg->lo, hi = pg->hi;
    int64_t r = writeback(c, *pg, k);
    if (r < 0) return r;
    pg->pristine = pg->data;  // the written-back state
    pg->dirty = true;         // still mapped writable: keep the range
    pg->lo = lo;
    pg->hi = hi;
  }
  return (int64_t)m;
}

// gfsync: write back every dirty page of the file.
ORC_API int orc_cache_fsync(void* h, int fd) {
  OCache* c = (OCache*)h;
  if (fd < 0 || (size_t)fd >= c->files.size() || c->files[fd].refs <= 0) return -EBADF;
  OFile& f = c->files[fd];
  for (auto& kv : c->pages) {
    if (kv.first.first != f.uid) continue;
    int64_t r = writeback(c, kv.second, kv.first);
    if (r < 0) return (int)r;
  }
  return 0;
}

// gftruncate (Tab.1; matvec output P:L1060): host ftruncate and
// reclaim cached pages wholly beyond the new size.
ORC_API int orc_cache_ftruncate(void* h, int fd, uint64_t size) {
  OCache* c = (OCache*)h;
  if (fd < 0 || (size_t)fd >= c->files.size() || c->files[fd].refs <= 0) return -EBADF;
  OFile& f = c->files[fd];
  if (ftruncate(f.hfd, (off_t)size) != 0) return -errno;
  std::vector<PKey> ks;
  for (auto& kv : c->pages)
    if (kv.first.first == f.uid && kv.first.second * c->P >= size) ks.push_back(kv.first);
  for (auto& k : ks) drop_page(c, k);
  f.size = size;
  return 0;
}

// counters: hits, misses, evictions, writebacks, resident pages
ORC_API void orc_cache_stats(void* h, uint64_t* out5) {
  OCache* c = (OCache*)h;
  out5[0] = c->hits;
  out5[1] = c->misses;
  out5[2] = c->evictions;
  out5[3] = c->writebacks;
  out5[4] = c->pages.size();
}

// ---------------------------------------------------------------------------
// O3 — grep -w (§5.2.2): "for each word in the dictionary, the
// program determines how many times and in which files it appears".
// Dictionary: one word per 32-byte slot; the file list is a
// file. Readings R10-R15 in DESIGN.md: word bytes [A-Za-z0-9_]
// (GNU grep -w under LC_ALL=C), counts per occurrence, dictionary words must be
// non-empty word-byte strings of <= 32 bytes, duplicate words allowed.
// ---------------------------------------------------------------------------
namespace {

inline bool is_word(uint8_t ch) {
  return (ch >= 'a' && ch <= 'z') || (ch >= 'A' && ch <= 'Z') || (ch >= '0' && ch <= '9') ||
         ch == '_';
}

inline uint64_t splitmix64(uint64_t x) {
  uint64_t z = x + 0x9E3779B97F4A7C15ull;
  z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
  return z ^ (z >> 31);
}

// Order-independent hit digest term for hit (file f, byte offset off, word k).
inline uint64_t hit_mix(uint64_t f, uint64_t off, uint64_t k) {
  return splitmix64(splitmix64(splitmix64(f) + off) + k);
}

int read_whole(const std::string& path, std::vector<uint8_t>* out) {
  int fd = open(path.c_str(), O_RDONLY);
  if (fd < 0) return -errno;
  struct stat st;
  if (fstat(fd, &st) != 0) { int e = -errno; close(fd); return e; }
  out->assign((size_t)st.st_size, 0);
  int64_t r = pread_full(fd, out->data(), (uint64_t)st.st_size, 0);
  close(fd);
  if (r < 0) return (int)r;
  out->resize((size_t)r);
  return 0;
}

int load_dict(const char* dict_path, std::vector<std::string>* words) {
  std::vector<uint8_t> d;
  int r = read_whole(dict_path, &d);
  if (r < 0) return r;
  if (d.size() % 32 != 0) return -EINVAL;
  for (size_t s = 0; s < d.size(); s += 32) {
    size_t n = strnlen((const char*)&d[s], 32);
    if (n == 0) return -EINVAL;
    for (size_t i = 0; i < n; ++i)
      if (!is_word(d[s + i])) return -EINVAL;
    words->emplace_back((const char*)&d[s], n);
  }
  return 0;
}

int load_list(const char* list_path, std::vector<std::string>* paths) {
  std::vector<uint8_t> d;
  int r = read_whole(list_path, &d);
  if (r < 0) return r;
  std::string dir(list_path);
  size_t slash = dir.rfind('/');
  dir = slash == std::string::npos ? std::string(".") : dir.substr(0, slash);
  size_t i = 0;
  while (i < d.size()) {
    size_t j = i;
    while (j < d.size() && d[j] != '\n') ++j;
    if (j > i) {
      std::string p((const char*)&d[i], j - i);
      if (p.size() >= 4096) return -ENAMETOOLONG;
      if (p[0] != '/') p = dir + "/" + p;
      paths->push_back(p);
    }
    i = j + 1;
  }
  return 0;
}

struct Hit {
  uint32_t f;
  uint64_t off;
  uint32_t k;
};

struct GrepResult {
  std::vector<uint32_t> rec_f, rec_k;
  std::vector<uint64_t> rec_c;
  std::vector<uint64_t> totals;
  uint64_t dig_sum = 0, dig_xor = 0, nhits = 0;
  std::vector<Hit> hits;
  uint64_t bytes = 0, nfiles = 0;
};

}  // namespace

// Tokenising oracle: scan left to right, tokens are maximal runs of word
// bytes, look each up in a hash map from word to dictionary indices.
ORC_API int orc_grep(const char* dict_path, const char* list_path, int want_hits, int nthreads,
                     void** out) {
  std::vector<std::string> words, paths;
  int r = load_dict(dict_path, &words);
  if (r < 0) return r;
  r = load_list(list_path, &paths);
  if (r < 0) return r;
  std::unordered_map<std::string, std::vector<uint32_t>> index;
  for (size_t k = 0; k < words.size(); ++k) index[words[k]].push_back((uint32_t)k);

  GrepResult* res = new GrepResult();
  res->totals.assign(words.size(), 0);
  res->nfiles = paths.size();
  if (nthreads < 1) nthreads = 1;
  std::vector<std::map<uint32_t, uint64_t>> per_file(paths.size());
  std::vector<std::vector<Hit>> per_file_hits(paths.size());
  std::vector<uint64_t> per_file_bytes(paths.size(), 0);
  std::vector<int> per_file_err(paths.size(), 0);

  auto work = [&](size_t t) {
    std::vector<uint8_t> text;
    for (size_t f = t; f < paths.size(); f += (size_t)nthreads) {
      int e = read_whole(paths[f], &text);
      if (e < 0) { per_file_err[f] = e; continue; }
      per_file_bytes[f] = text.size();
      size_t L = text.size(), i = 0;
      while (i < L) {
        if (!is_word(text[i])) { ++i; continue; }
        size_t s = i;
        while (i < L && is_word(text[i])) ++i;
        size_t n = i - s;
        if (n > 32) continue;
        auto it = index.find(std::string((const char*)&text[s], n));
        if (it == index.end()) continue;
        for (uint32_t k : it->second) {
          per_file[f][k] += 1;
          per_file_hits[f].push_back(Hit{(uint32_t)f, (uint64_t)s, k});
        }
      }
    }
  };
  std::vector<std::thread> th;
  for (int t = 0; t < nthreads; ++t) th.emplace_back(work, (size_t)t);
  for (auto& x : th) x.join();
  for (size_t f = 0; f < paths.size(); ++f) {
    if (per_file_err[f]) { int e = per_file_err[f]; delete res; return e; }
    res->bytes += per_file_bytes[f];
    for (auto& kv : per_file[f]) {  // std::map: sorted by word index
      res->rec_f.push_back((uint32_t)f);
      res->rec_k.push_back(kv.first);
      res->rec_c.push_back(kv.second);
      res->totals[kv.first] += kv.second;
    }
    for (auto& hh : per_file_hits[f]) {
      uint64_t m = hit_mix(hh.f, hh.off, hh.k);
      res->dig_sum += m;
      res->dig_xor ^= m;
      res->nhits++;
    }
    if (want_hits) {
      std::sort(per_file_hits[f].begin(), per_file_hits[f].end(), [](const Hit& a, const Hit& b) {
        return a.off != b.off ? a.off < b.off : a.k < b.k;
      });
      res->hits.insert(res->hits.end(), per_file_hits[f].begin(), per_file_hits[f].end());
    }
  }
  *out = res;
  return 0;
}

// Brute force (pin for orc_grep): the literal grep -w definition per
// occurrence — cnt[f][k] = #{ i : t[i..i+|w|) = w, (i = 0 or not W(t[i-1])),
// (i+|w| = L or not W(t[i+|w|])) } — one dictionary word at a time, the way
// the paper's kernel assigns one word per thread.
ORC_API int orc_grep_brute(const char* dict_path, const char* list_path, void** out) {
  std::vector<std::string> words, paths;
  int r = load_dict(dict_path, &words);
  if (r < 0) return r;
  r = load_list(list_path, &paths);
  if (r < 0) return r;
  GrepResult* res = new GrepResult();
  res->totals.assign(words.size(), 0);
  res->nfiles = paths.size();
  std::vector<uint8_t> t;
  for (size_t f = 0; f < paths.size(); ++f) {
    int e = read_whole(paths[f], &t);
    if (e < 0) { delete res; return e; }
    res->bytes += t.size();
    size_t L = t.size();
    std::vector<Hit> fh;
    for (size_t k = 0; k < words.size(); ++k) {
      const std::string& w = words[k];
      size_t n = w.size();
      uint64_t cnt = 0;
      for (size_t i = 0; i + n <= L; ++i) {
        if (memcmp(&t[i], w.data(), n) != 0) continue;
        if (i > 0 && is_word(t[i - 1])) continue;
        if (i + n < L && is_word(t[i + n])) continue;
        cnt++;
        fh.push_back(Hit{(uint32_t)f, (uint64_t)i, (uint32_t)k});
      }
      if (cnt) {
        res->rec_f.push_back((uint32_t)f);
        res->rec_k.push_back((uint32_t)k);
        res->rec_c.push_back(cnt);
        res->totals[k] += cnt;
      }
    }
    for (auto& hh : fh) {
      uint64_t m = hit_mix(hh.f, hh.off, hh.k);
      res->dig_sum += m;
      res->dig_xor ^= m;
      res->nhits++;
    }
    std::sort(fh.begin(), fh.end(), [](const Hit& a, const Hit& b) {
      return a.off != b.off ? a.off < b.off : a.k < b.k;
    });
    res->hits.insert(res->hits.end(), fh.begin(), fh.end());
  }
  *out = res;
  return 0;
}

// Accessors. counts[0..5] = nrecords, nwords, nhits, listed hits, bytes, nfiles.
ORC_API void orc_grep_counts(void* h, uint64_t* c6) {
  GrepResult* r = (GrepResult*)h;
  c6[0] = r->rec_f.size();
  c6[1] = r->totals.size();
  c6[2] = r->nhits;
  c6[3] = r->hits.size();
  c6[4] = r->bytes;
  c6[5] = r->nfiles;
}

ORC_API void orc_grep_get(void* h, uint32_t* rec_f, uint32_t* rec_k, uint64_t* rec_c,
                          uint64_t* totals, uint64_t* digest2, uint32_t* hit_f, uint64_t* hit_off,
                          uint32_t* hit_k) {
  GrepResult* r = (GrepResult*)h;
  for (size_t i = 0; i < r->rec_f.size(); ++i) {
    if (rec_f) rec_f[i] = r->rec_f[i];
    if (rec_k) rec_k[i] = r->rec_k[i];
    if (rec_c) rec_c[i] = r->rec_c[i];
  }
  if (totals)
    for (size_t k = 0; k < r->totals.size(); ++k) totals[k] = r->totals[k];
  if (digest2) {
    digest2[0] = r->dig_sum;
    digest2[1] = r->dig_xor;
  }
  for (size_t i = 0; i < r->hits.size(); ++i) {
    if (hit_f) hit_f[i] = r->hits[i].f;
    if (hit_off) hit_off[i] = r->hits[i].off;
    if (hit_k) hit_k[i] = r->hits[i].k;
  }
}

ORC_API void orc_grep_free(void* h) { delete (GrepResult*)h; }

// ---------------------------------------------------------------------------
// O4 — matrix-vector product (§5.1.4): y_r = sum_j A_rj x_j with
// A read from a row-major little-endian fp32 file, accumulated in float64
// (R16), then reported in float64 (the caller rounds to fp32).
// ---------------------------------------------------------------------------
ORC_API int orc_matvec(const char* a_path, const char* x_path, uint64_t rows, uint64_t cols,
                       uint64_t row0, uint64_t nrows, int nthreads, double* y) {
  std::vector<float> x(cols);
  {
    int fd = open(x_path, O_RDONLY);
    if (fd < 0) return -errno;
    int64_t r = pread_full(fd, (uint8_t*)x.data(), cols * 4, 0);
    close(fd);
    if (r < 0) return (int)r;
    if ((uint64_t)r != cols * 4) return -EIO;
  }
  if (row0 + nrows > rows) return -EINVAL;
  if (nthreads < 1) nthreads = 1;
  std::vector<int> errs(nthreads, 0);
  auto work = [&](int t) {
    int fd = open(a_path, O_RDONLY);
    if (fd < 0) { errs[t] = -errno; return; }
    std::vector<float> row(cols);
    for (uint64_t i = row0 + t; i < row0 + nrows; i += nthreads) {
      int64_t r = pread_full(fd, (uint8_t*)row.data(), cols * 4, i * cols * 4);
      if (r < 0 || (uint64_t)r != cols * 4) { errs[t] = r < 0 ? (int)r : -EIO; break; }
      double acc = 0.0;
      for (uint64_t j = 0; j < cols; ++j) acc += (double)row[j] * (double)x[j];
      y[i - row0] = acc;
    }
    close(fd);
  };
  std::vector<std::thread> th;
  for (int t = 0; t < nthreads; ++t) th.emplace_back(work, t);
  for (auto& z : th) z.join();
  for (int e : errs)
    if (e) return e;
  return 0;
}
