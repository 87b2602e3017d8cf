// gfs_grep.cu — exact whole-word string search (grep -w) over many files,
// built on the GPUfs device API (§5.2.2).
//
// Problem statement: for each dictionary word, how many times
// and in which files it appears. Dictionary: one word per 32-byte slot
// (P:L1264-1266). The list of input files is itself read from a file
// (P:L1266-1267). Every file byte reaches the kernels through gopen/gread.
//
// The paper assigns one dictionary word per thread and brute-forces every
// position. Here the result is the same (pinned
// against the brute-force oracle) but the work is proportional to the corpus:
//   k_grep_dict   gread the dictionary, validate slots, build an open-addressing
//                 hash table (L2-resident) keyed by a 64-bit token hash;
//   k_grep_list_* gread the file list in chunks, count line starts per chunk,
//                 scan, emit absolute paths (parallel over the list);
//   k_grep_open   gopen every file once (first gopen goes to the host,
//                 P:L370-372), record fd and size;
//   k_grep_plan   exclusive scan of per-file work-item counts, item -> file map;
//   k_grep_scan   persistent blocks pull items: a whole file when it fits one
//                 item, else a chunk of it. gread brings the item plus a halo
//                 into shared memory (TMA). Pass 1 classifies 32-byte stripes
//                 into word-byte bit masks (SWAR, 4 bytes per op); pass 2 gives
//                 each thread the tokens that start in its stripe: length from
//                 the masks, bytes gathered as 8 zero-padded words, one 64-bit
//                 hash, one probe of the (L2-resident) table, an exact 32-byte
//                 compare on a fingerprint match. Counts per item in shared
//                 memory; a whole-file item emits its (file, word, count)
//                 records directly, chunks of large files merge through a
//                 global (file, word) table;
//   k_grep_close  gclose every file (unless kept open for warm re-runs);
//   k_grep_compact emit unique (file, word, count) records and word totals.
// Word bytes are [A-Za-z0-9_] (GNU grep -w under LC_ALL=C, R10).
#include <cuda_runtime.h>
#include <errno.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>
#include <time.h>

#include "gpufs.h"
#include "gpufs_device.cuh"

#define GFS_API extern "C" __attribute__((visibility("default")))

using namespace gfs;

namespace {

constexpr uint32_t kMaxPath = GFS_MAX_PATH;
constexpr uint32_t kHalo = 48;      // bytes after the chunk: a token starting inside may run 33 bytes
constexpr uint32_t kPre = 16;       // bytes before the chunk (one needed for the boundary test)
constexpr uint32_t kSlack = 64;     // gathers read up to 48 bytes past a token start
constexpr uint32_t kCountSlots = 2048;
constexpr uint32_t kListRead = 65536;  // list file gread granularity
constexpr uint32_t kListChunk = 4096;  // list parse granularity (one block per chunk)
constexpr uint64_t kPairEmpty = ~0ull;
constexpr uint64_t kDupBit = 1ull << 63;  // table entry: the word has duplicates

struct GrepWork {
  // dictionary
  uint8_t* dict;          // max_words * 32
  uint64_t* table;        // (dup << 63) | (fp31 << 32) | (len << 26) | (k + 1); 0 = empty
  uint32_t table_mask;
  uint32_t* dup_head;     // per primary word: first duplicate + 1
  uint32_t* dup_next;     // per word: next duplicate + 1
  // file list
  uint8_t* list;          // list_cap bytes
  uint32_t* list_chunk;   // per list chunk: line starts (then exclusive prefix)
  char* paths;            // max_files * kMaxPath
  int32_t* fd;
  uint64_t* size;
  uint64_t* item_base;    // max_files + 1
  uint32_t* item_file;    // item -> file
  uint64_t max_items;
  // (file, word) -> count table
  uint64_t* pair;         // slot i: pair[2i] = (file << 32) | word (or empty), pair[2i+1] = count;
                          // key and count share one 32-byte sector
  uint64_t pair_mask;
  // counters
  unsigned long long* vars;  // see V_*
  unsigned long long* prof;  // GFS_GREP_PROF=1: per-phase cycles of k_grep_scan thread 0 (else null)
};
enum { V_NFILES = 0, V_NWORDS, V_NITEMS, V_NEXT, V_ERR, V_BYTES, V_NREC, V_NHITS, V_DSUM, V_DXOR, V_NLISTED,
       V_NEXTF, V_LISTSZ, V_HOLD_DICT, V_HOLD_LIST, V_NVARS };

__device__ __forceinline__ bool is_word(uint32_t ch) {
  return (ch - 'a' < 26u) || (ch - 'A' < 26u) || (ch - '0' < 10u) || ch == '_';
}

// Word-byte mask of 4 bytes (SWAR): bit 7 of each byte set iff it is in
// [A-Za-z0-9_]. in_range(x, lo, hi) per byte for x, lo, hi <= 0x7f:
// (0x80 + x - lo) has bit 7 iff x >= lo, (0x80 + hi - x) iff x <= hi, and
// neither subtraction borrows across bytes. Bytes >= 0x80 are non-word.
__device__ __forceinline__ uint32_t word_bits4(uint32_t x) {
  constexpr uint32_t H = 0x80808080u, O = 0x01010101u;
  const uint32_t x7 = x & 0x7F7F7F7Fu;
  const uint32_t l = x7 | 0x20202020u;  // fold A-Z onto a-z
  const uint32_t alpha = ((l | H) - 0x61u * O) & ((0x7Au | 0x80u) * O - l);
  const uint32_t digit = ((x7 | H) - 0x30u * O) & ((0x39u | 0x80u) * O - x7);
  const uint32_t under = ((x7 | H) - 0x5Fu * O) & ((0x5Fu | 0x80u) * O - x7);
  const uint32_t m = (alpha | digit | under) & ~x & H;
  // bits 7,15,23,31 -> 0..3 (the four partial products never overlap)
  return (((m >> 7) * 0x00204081u) >> 21) & 0xFu;
}

// 32-bit word-byte mask of 32 bytes at p (16-byte aligned shared memory).
__device__ __forceinline__ uint32_t word_bits32(const uint8_t* p) {
  const uint4 a = *(const uint4*)p, b = *(const uint4*)(p + 16);
  return word_bits4(a.x) | (word_bits4(a.y) << 4) | (word_bits4(a.z) << 8) | (word_bits4(a.w) << 12) |
         (word_bits4(b.x) << 16) | (word_bits4(b.y) << 20) | (word_bits4(b.z) << 24) | (word_bits4(b.w) << 28);
}

// Hash of a word from its first 8 bytes (zero-padded past its length L) and
// L. Longer words sharing a prefix and length collide on purpose: every key
// match is confirmed by an exact 32-byte compare, and the table keeps each
// such word in its own entry (k_grep_dict), so lookups stay exact.
__device__ __forceinline__ uint64_t tok_hash(uint32_t w0, uint32_t w1, uint32_t L) {
  uint64_t h = (((uint64_t)w1 << 32) | w0) ^ (0x9E3779B97F4A7C15ull * L);
  h *= 0xBF58476D1CE4E5B9ull;
  h ^= h >> 29;
  h *= 0x94D049BB133111EBull;
  return h ^ (h >> 32);
}

// Low `nb` (0..4) bytes of a word.
__device__ __forceinline__ uint32_t low_bytes(uint32_t x, int nb) {
  return x & __funnelshift_lc(0xFFFFFFFFu, 0u, 8 * nb);
}

// Bytes [0, L) of the 32 starting at byte offset `sh` (0..15) of 12 words,
// as 8 zero-padded words: two select levels + a funnel shift, no local memory.
__device__ __forceinline__ void gather_token(const uint32_t (&W)[12], uint32_t sh, uint32_t L, uint32_t (&v)[8]) {
  uint32_t A[10], B[9];
#pragma unroll
  for (int j = 0; j < 10; ++j) A[j] = (sh & 8) ? W[j + 2] : W[j];
#pragma unroll
  for (int j = 0; j < 9; ++j) B[j] = (sh & 4) ? A[j + 1] : A[j];
  const uint32_t r = (sh & 3) * 8;
#pragma unroll
  for (int j = 0; j < 8; ++j) {
    const uint32_t wv = __funnelshift_r(B[j], B[j + 1], r);
    const int nb = min(max((int)L - 4 * j, 0), 4);
    v[j] = wv & __funnelshift_lc(0xFFFFFFFFu, 0u, 8 * nb);  // low nb bytes
  }
}

// entry bits 32..62 hold a 31-bit fingerprint, 26..31 the length
__device__ __forceinline__ uint64_t entry_key(uint64_t h, uint32_t len) {
  return (((h >> 33) & 0x7FFFFFFFull) << 32) | ((uint64_t)len << 26);
}
__device__ __forceinline__ uint64_t key_bits(uint64_t e) { return (e & ~kDupBit) >> 26; }

__device__ __forceinline__ uint64_t splitmix64(uint64_t x) {
  uint64_t z = x + 0x9E3779B97F4A7C15ull;
  z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
  return z ^ (z >> 31);
}

// Order-independent digest term of one hit (file f, byte offset off, word k).
// The digest term of one hit (R20); hit_mix_hf below is the form the scan uses.
__device__ __forceinline__ __attribute__((unused)) uint64_t hit_mix(uint64_t f, uint64_t off, uint64_t k) {
  return splitmix64(splitmix64(splitmix64(f) + off) + k);
}
// The same with splitmix64(f) computed once per file (hf).
__device__ __forceinline__ uint64_t hit_mix_hf(uint64_t hf, uint64_t off, uint64_t k) {
  return splitmix64(splitmix64(hf + off) + k);
}

__device__ __forceinline__ void set_err(GrepWork& w, long long e) { atomicMin((long long*)&w.vars[V_ERR], e); }

// --------------------------------------------------------------- hold
// One block opens the dictionary and the list before the blocks that read
// them and closes them after the run: the many short gopen/gclose pairs of
// the reading blocks then never drop the count to zero, which would make the
// next opener re-validate the file with the host (close-to-open).
__global__ void k_grep_hold(const gfs_ctx* c, const char* dict_path, const char* list_path, GrepWork w, int release) {
  if (!release) {
    const int a = gopen(c, dict_path, GFS_O_RDONLY);
    const int b = gopen(c, list_path, GFS_O_RDONLY);
    if (threadIdx.x == 0) {
      w.vars[V_HOLD_DICT] = (unsigned long long)(long long)a;
      w.vars[V_HOLD_LIST] = (unsigned long long)(long long)b;
    }
  } else {
    const int a = (int)(long long)w.vars[V_HOLD_DICT], b = (int)(long long)w.vars[V_HOLD_LIST];
    if (a >= 0) gclose(c, a);
    if (b >= 0) gclose(c, b);
  }
}

// --------------------------------------------------------------- dictionary
__global__ void k_grep_dict(const gfs_ctx* c, const char* dict_path, GrepWork w, uint32_t max_words) {
  const int tid = threadIdx.x;
  const int fd = gopen(c, dict_path, GFS_O_RDONLY);
  if (fd < 0) {
    if (tid == 0 && blockIdx.x == 0) set_err(w, fd);
    return;
  }
  const int64_t size = gfstat_size(c, fd);
  if (size % 32 != 0 || size / 32 > (int64_t)max_words) {
    if (tid == 0 && blockIdx.x == 0) set_err(w, size % 32 ? -EINVAL : -ENOSPC);
    gclose(c, fd);
    return;
  }
  const uint32_t N = (uint32_t)(size / 32);
  if (blockIdx.x == 0 && tid == 0) w.vars[V_NWORDS] = N;
  // each block reads a contiguous slice of slots, then inserts those words
  const uint32_t per = (N + gridDim.x - 1) / gridDim.x;
  const uint32_t k0 = blockIdx.x * per, k1 = min(N, k0 + per);
  if (k0 < k1) {
    const int64_t r = gread(c, fd, (uint64_t)k0 * 32, (uint64_t)(k1 - k0) * 32, w.dict + (size_t)k0 * 32);
    __threadfence();  // this block's dictionary bytes are visible before its table entries
    if (r != (int64_t)(k1 - k0) * 32) {
      if (tid == 0) set_err(w, r < 0 ? r : -EIO);
    } else {
      for (uint32_t k = k0 + tid; k < k1; k += blockDim.x) {
        uint8_t* s = w.dict + (size_t)k * 32;
        uint32_t n = 0;
        while (n < 32 && s[n]) ++n;
        bool ok = n > 0;
        for (uint32_t i = 0; i < n; ++i) ok &= is_word(s[i]);
        if (!ok) {  // empty slot or non-word byte (R13)
          set_err(w, -EINVAL);
          continue;
        }
        // zero the bytes after the word: the slot becomes the word's padded form
        // (other threads only ever read bytes [0, n) of a slot of length n)
        for (uint32_t i = n; i < 32; ++i) s[i] = 0;
        const uint64_t h = tok_hash(((const uint32_t*)s)[0], ((const uint32_t*)s)[1], n);
        const uint64_t ent = entry_key(h, n) | (k + 1);
        // linear probing from the start of the hash's 4-entry (32-byte) bucket:
        // lookups read a whole bucket per step (scan_token)
        uint32_t slot = (uint32_t)h & w.table_mask & ~3u;
        for (uint32_t probe = 0; probe <= w.table_mask; ++probe, slot = (slot + 1) & w.table_mask) {
          unsigned long long cur = atomicCAS((unsigned long long*)&w.table[slot], 0ull, (unsigned long long)ent);
          if (cur == 0) break;
          if (key_bits(cur) == key_bits(ent)) {  // same fingerprint and length: same word?
            const uint32_t kp = (uint32_t)(cur & ((1u << 26) - 1)) - 1;
            const uint8_t* t = w.dict + (size_t)kp * 32;
            bool same = true;
            for (uint32_t i = 0; i < n; ++i) same &= t[i] == s[i];
            if (same) {  // duplicate dictionary word: chain it behind kp, flag the entry
              w.dup_next[k] = atomicExch(&w.dup_head[kp], k + 1);
              atomicOr((unsigned long long*)&w.table[slot], (unsigned long long)kDupBit);
              break;
            }
          }
        }
      }
    }
  }
  gclose(c, fd);
}

// --------------------------------------------------------------- file list
// Pass 1: every block greads its 64 KiB pieces of the list file.
__global__ void k_grep_list_read(const gfs_ctx* c, const char* list_path, GrepWork w, uint64_t list_cap) {
  const int fd = gopen(c, list_path, GFS_O_RDONLY);
  if (fd < 0) {
    if (threadIdx.x == 0 && blockIdx.x == 0) set_err(w, fd);
    return;
  }
  const int64_t size = gfstat_size(c, fd);
  if (size > (int64_t)list_cap) {
    if (threadIdx.x == 0 && blockIdx.x == 0) set_err(w, -ENOSPC);
  } else {
    if (threadIdx.x == 0 && blockIdx.x == 0) w.vars[V_LISTSZ] = (unsigned long long)size;
    for (uint64_t o = (uint64_t)blockIdx.x * kListRead; o < (uint64_t)size; o += (uint64_t)gridDim.x * kListRead) {
      const uint64_t n = min((uint64_t)kListRead, (uint64_t)size - o);
      const int64_t r = gread(c, fd, o, n, w.list + o);
      if (r != (int64_t)n && threadIdx.x == 0) set_err(w, r < 0 ? r : -EIO);
    }
  }
  gclose(c, fd);
}

__device__ __forceinline__ bool line_start(const uint8_t* L, uint64_t i) {
  return L[i] != '\n' && (i == 0 || L[i - 1] == '\n');
}

// Pass 2: line starts (non-empty lines) per chunk.
__global__ void k_grep_list_count(GrepWork w) {
  __shared__ uint32_t cnt_s;
  const uint64_t size = w.vars[V_LISTSZ];
  const uint64_t nch = (size + kListChunk - 1) / kListChunk;
  for (uint64_t ch = blockIdx.x; ch < nch; ch += gridDim.x) {
    if (threadIdx.x == 0) cnt_s = 0;
    __syncthreads();
    const uint64_t a = ch * kListChunk, b = min(size, a + kListChunk);
    uint32_t n = 0;
    for (uint64_t i = a + threadIdx.x; i < b; i += blockDim.x) n += line_start(w.list, i);
    atomicAdd(&cnt_s, n);
    __syncthreads();
    if (threadIdx.x == 0) w.list_chunk[ch] = cnt_s;
    __syncthreads();
  }
}

// Pass 3 (one block): exclusive scan of the chunk counts.
__global__ void k_grep_list_scan(GrepWork w, uint32_t max_files) {
  if (threadIdx.x != 0) return;
  const uint64_t size = w.vars[V_LISTSZ];
  const uint64_t nch = (size + kListChunk - 1) / kListChunk;
  uint32_t run = 0;
  for (uint64_t ch = 0; ch < nch; ++ch) {
    const uint32_t v = w.list_chunk[ch];
    w.list_chunk[ch] = run;
    run += v;
  }
  if (run > max_files) set_err(w, -ENOSPC);
  w.vars[V_NFILES] = run < max_files ? run : max_files;
}

// Pass 4: each line start writes its absolute path (relative paths resolve
// against the list file's directory, R15).
__global__ void k_grep_list_emit(GrepWork w, const char* dir, uint32_t dir_len, uint32_t max_files) {
  __shared__ uint32_t warp_tot[32];
  __shared__ uint32_t base_s;
  const uint64_t size = w.vars[V_LISTSZ];
  const uint64_t nch = (size + kListChunk - 1) / kListChunk;
  const int tid = threadIdx.x, lane = tid & 31, wid = tid >> 5, nw = (blockDim.x + 31) / 32;
  const uint8_t* L = w.list;
  for (uint64_t ch = blockIdx.x; ch < nch; ch += gridDim.x) {
    if (tid == 0) base_s = w.list_chunk[ch];
    __syncthreads();
    const uint64_t a = ch * kListChunk, b = min(size, a + kListChunk);
    for (uint64_t t0 = a; t0 < b; t0 += blockDim.x) {
      const uint64_t i = t0 + tid;
      const bool start = i < b && line_start(L, i);
      const uint32_t bal = __ballot_sync(0xFFFFFFFFu, start);
      if (lane == 0) warp_tot[wid] = __popc(bal);
      __syncthreads();
      uint32_t k = base_s;
      for (int q = 0; q < wid; ++q) k += warp_tot[q];
      k += __popc(bal & ((1u << lane) - 1));
      if (start && k < max_files) {
        uint32_t n = 0;
        while (i + n < size && L[i + n] != '\n') ++n;
        char* dst = w.paths + (size_t)k * kMaxPath;
        uint32_t o = 0;
        if (L[i] != '/') {
          for (uint32_t q = 0; q < dir_len && o < kMaxPath - 1; ++q) dst[o++] = dir[q];
          if (o < kMaxPath - 1) dst[o++] = '/';
        }
        if (o + n >= kMaxPath) {
          set_err(w, -ENAMETOOLONG);
          n = 0;
        }
        for (uint32_t q = 0; q < n; ++q) dst[o + q] = (char)L[i + q];
        dst[o + n] = 0;
      }
      __syncthreads();
      if (tid == 0) {
        uint32_t tot = 0;
        for (int q = 0; q < nw; ++q) tot += warp_tot[q];
        base_s += tot;
      }
      __syncthreads();
    }
  }
}

// --------------------------------------------------------------- open files
__global__ void k_grep_open(const gfs_ctx* c, GrepWork w, uint32_t chunk) {
  __shared__ uint32_t f_s;
  const int tid = threadIdx.x;
  const uint32_t nfiles = (uint32_t)w.vars[V_NFILES];
  for (;;) {
    if (tid == 0) f_s = (uint32_t)atomicAdd(&w.vars[V_NEXTF], 1ull);
    __syncthreads();
    const uint32_t f = f_s;
    if (f >= nfiles) break;
    // first gopen of a file goes to the host; page 0 comes back with it
    const int fd = gopen(c, w.paths + (size_t)f * kMaxPath, GFS_O_RDONLY | GFS_O_PREFETCH);
    const int64_t sz = fd >= 0 ? gfstat_size(c, fd) : fd;
    if (tid == 0) {
      w.fd[f] = fd;
      if (sz < 0) {
        set_err(w, sz);
        w.size[f] = 0;
        w.item_base[f] = 0;
      } else {
        w.size[f] = (uint64_t)sz;
        w.item_base[f] = ((uint64_t)sz + chunk - 1) / chunk;  // item count; scanned later
        atomicAdd(&w.vars[V_BYTES], (unsigned long long)sz);
      }
    }
    __syncthreads();
  }
}

// exclusive scan of item counts -> item_base, one block
__global__ void k_grep_plan(GrepWork w) {
  __shared__ uint64_t part[1024];
  const int tid = threadIdx.x, nthr = blockDim.x;
  const uint32_t n = (uint32_t)w.vars[V_NFILES];
  const uint32_t per = (n + nthr - 1) / nthr;
  const uint32_t a = tid * per, b = min(n, a + per);
  uint64_t s = 0;
  for (uint32_t i = a; i < b; ++i) s += w.item_base[i];
  part[tid] = s;
  __syncthreads();
  if (tid == 0) {
    uint64_t run = 0;
    for (int q = 0; q < nthr; ++q) {
      const uint64_t v = part[q];
      part[q] = run;
      run += v;
    }
    if (run > w.max_items) {
      set_err(w, -ENOSPC);
      run = w.max_items;
    }
    w.vars[V_NITEMS] = run;
    w.item_base[n] = run;
  }
  __syncthreads();
  uint64_t run = part[tid];
  for (uint32_t i = a; i < b; ++i) {
    const uint64_t v = w.item_base[i];
    w.item_base[i] = run;
    run += v;
  }
}

// item -> file map (one thread per file)
__global__ void k_grep_items(GrepWork w) {
  const uint32_t n = (uint32_t)w.vars[V_NFILES];
  for (uint32_t f = blockIdx.x * blockDim.x + threadIdx.x; f < n; f += gridDim.x * blockDim.x) {
    const uint64_t a = w.item_base[f], b = min(w.item_base[f + 1], w.max_items);
    for (uint64_t i = a; i < b; ++i) w.item_file[i] = f;
  }
}

// --------------------------------------------------------------- scan
__device__ __forceinline__ void pair_add(GrepWork& w, uint32_t f, uint32_t k, uint64_t cnt) {
  const uint64_t key = ((uint64_t)f << 32) | k;
  uint64_t slot = splitmix64(key) & w.pair_mask;
  for (uint64_t probe = 0; probe <= w.pair_mask; ++probe, slot = (slot + 1) & w.pair_mask) {
    unsigned long long cur = atomicCAS((unsigned long long*)&w.pair[2 * slot], (unsigned long long)kPairEmpty,
                                       (unsigned long long)key);
    if (cur == kPairEmpty || cur == key) {
      atomicAdd((unsigned long long*)&w.pair[2 * slot + 1], (unsigned long long)cnt);
      return;
    }
  }
  set_err(w, -ENOSPC);
}

struct ScanAcc {
  uint64_t dsum, dxor, nh;
};

// Shared-memory state of one scan block (dynamic shared memory, see scan_smem).
struct ScanSmem {
  uint8_t* buf;     // kPre + chunk + kHalo + kSlack bytes; file byte p at buf[kPre + p - s]
  uint32_t* mask;   // word-byte bits per 32-byte stripe of buf (+1 zero stripe)
  uint32_t* ckey;   // count table: word + 1 (0 = empty)
  uint32_t* ccnt;
  uint16_t* olist;  // occupied count slots, in insertion order
  uint64_t hf;      // splitmix64(file index) of the current item (digest)
  uint32_t cmask;   // count table slots - 1
};

// One hit of word k at file position pos: per-item shared count (spilling to
// the global table when the probe run is exhausted), digest, optional hit list.
__device__ __forceinline__ void count_hit(GrepWork& w, const ScanSmem& S, uint32_t* nocc, uint32_t* spilled,
                                          uint32_t f, uint32_t k, uint64_t pos, uint64_t* hits, uint64_t hit_cap,
                                          ScanAcc& acc) {
  uint32_t cs = (k * 2654435761u) & S.cmask;
  bool done = false;
  for (uint32_t p = 0; p < 64; ++p, cs = (cs + 1) & S.cmask) {
    const uint32_t prev = atomicCAS(&S.ckey[cs], 0u, k + 1);
    if (prev == 0) S.olist[atomicAdd(nocc, 1u)] = (uint16_t)cs;
    if (prev == 0 || prev == k + 1) {
      atomicAdd(&S.ccnt[cs], 1u);
      done = true;
      break;
    }
  }
  if (!done) {  // this item's records then all go through the global table
    pair_add(w, f, k, 1);
    *spilled = 1;
  }
  const uint64_t m = hit_mix_hf(S.hf, pos, k);
  acc.dsum += m;
  acc.dxor ^= m;
  ++acc.nh;
  if (hits) {
    const unsigned long long idx = atomicAdd(&w.vars[V_NLISTED], 1ull);
    if (idx < hit_cap) {
      hits[2 * idx] = ((uint64_t)f << 32) | k;
      hits[2 * idx + 1] = pos;
    }
  }
}

// One token: bytes buf[i, i + L), file position pos, 1 <= L <= 32.
__device__ __forceinline__ void scan_token(GrepWork& w, const ScanSmem& S, uint32_t* nocc, uint32_t* spilled,
                                           uint32_t f, uint32_t i, uint32_t L, uint64_t pos, uint64_t* hits,
                                           uint64_t hit_cap, ScanAcc& acc) {
  // first 8 bytes: three aligned words and two funnel shifts
  const uint32_t* a = (const uint32_t*)(S.buf + (i & ~3u));
  const uint32_t a0 = a[0], a1 = a[1], a2 = a[2], r8 = (i & 3u) * 8;
  const uint32_t w0 = low_bytes(__funnelshift_r(a0, a1, r8), min((int)L, 4));
  const uint32_t w1 = low_bytes(__funnelshift_r(a1, a2, r8), min(max((int)L - 4, 0), 4));
  const uint64_t h = tok_hash(w0, w1, L);
  const uint64_t want = entry_key(h, L) >> 26;
  // One 32-byte bucket (4 entries) per step; insertion filled the first empty
  // slot in the same order, so an empty slot ends the search.
  uint32_t b = (uint32_t)h & w.table_mask & ~3u;
  for (;;) {
    const uint4* bp = (const uint4*)&w.table[b];
    const uint4 e01 = __ldg(bp), e23 = __ldg(bp + 1);
    const uint64_t ent[4] = {((uint64_t)e01.y << 32) | e01.x, ((uint64_t)e01.w << 32) | e01.z,
                             ((uint64_t)e23.y << 32) | e23.x, ((uint64_t)e23.w << 32) | e23.z};
    bool empty = false;
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      empty |= ent[q] == 0;
      if (ent[q] != 0 && key_bits(ent[q]) == want) {
        const uint32_t kp = (uint32_t)(ent[q] & ((1u << 26) - 1)) - 1;
        const uint4* dw = (const uint4*)(w.dict + (size_t)kp * 32);  // padded slot (k_grep_dict)
        const uint4 d0 = __ldg(dw), d1 = __ldg(dw + 1);
        uint32_t v[8];  // the whole token, zero-padded: only gathered on a key match
        {
          uint32_t W[12];
          const uint4* qv = (const uint4*)(S.buf + (i & ~15u));
#pragma unroll
          for (int j = 0; j < 3; ++j) {
            const uint4 t = qv[j];
            W[4 * j] = t.x;
            W[4 * j + 1] = t.y;
            W[4 * j + 2] = t.z;
            W[4 * j + 3] = t.w;
          }
          gather_token(W, i & 15u, L, v);
        }
        const bool same = ((d0.x ^ v[0]) | (d0.y ^ v[1]) | (d0.z ^ v[2]) | (d0.w ^ v[3]) | (d1.x ^ v[4]) |
                           (d1.y ^ v[5]) | (d1.z ^ v[6]) | (d1.w ^ v[7])) == 0;
        if (same) {
          count_hit(w, S, nocc, spilled, f, kp, pos, hits, hit_cap, acc);
          if (ent[q] & kDupBit) {  // the word's duplicates each count (R14)
            for (uint32_t d = w.dup_head[kp]; d; d = w.dup_next[d - 1])
              count_hit(w, S, nocc, spilled, f, d - 1, pos, hits, hit_cap, acc);
          }
          return;
        }
      }
    }
    if (empty) return;
    b = (b + 4) & w.table_mask;
  }
}

// Bits [lo, hi) of a 32-bit mask (lo, hi clamped to [0, 32]).
__device__ __forceinline__ uint32_t bit_range(int lo, int hi) {
  lo = min(max(lo, 0), 32);
  hi = min(max(hi, 0), 32);
  if (hi <= lo) return 0u;
  const uint32_t upto_hi = hi == 32 ? 0xFFFFFFFFu : ((1u << hi) - 1u);
  const uint32_t below_lo = lo == 32 ? 0xFFFFFFFFu : ((1u << lo) - 1u);
  return upto_hi & ~below_lo;
}

__global__ void __launch_bounds__(256, 3) k_grep_scan(const gfs_ctx* c, GrepWork w, uint32_t chunk, uint64_t* hits,
                                                   uint64_t hit_cap, uint64_t* totals, uint32_t* rec,
                                                   uint64_t rec_cap) {
  extern __shared__ __align__(16) uint8_t sm[];
  const int tid = threadIdx.x, nthr = blockDim.x, lane = tid & 31, wid = tid >> 5;
  const uint32_t buf_bytes = (kPre + chunk + kHalo + kSlack + 15) & ~15u;
  const uint32_t nstripe_max = (kPre + chunk + kHalo + 31) / 32;
  ScanSmem S;
  S.buf = sm;
  S.mask = (uint32_t*)(sm + buf_bytes);
  S.ckey = S.mask + ((nstripe_max + 1 + 3) & ~3u);
  S.ccnt = S.ckey + kCountSlots;
  S.olist = (uint16_t*)(S.ccnt + kCountSlots);
  S.cmask = kCountSlots - 1;
  uint16_t* tok = S.olist + kCountSlots;  // token starts of one round: <= 32 per thread
  const uint32_t round_stripes = 2u * (uint32_t)nthr;
  __shared__ uint64_t nxt_item, nxt_size, nxt_base;
  __shared__ uint32_t nxt_f;
  __shared__ int32_t nxt_fd;
  __shared__ uint32_t nocc_s, spilled_s;
  __shared__ uint32_t warp_tot[32];
  __shared__ unsigned long long rbase_s;
  const uint64_t nitems = w.vars[V_NITEMS];
  ScanAcc acc{0, 0, 0};
  // tid 0 claims the next item and loads its file fields while the block
  // works on the current one (three dependent L2 round trips off the path)
  auto prefetch = [&]() {
    const uint64_t it = atomicAdd(&w.vars[V_NEXT], 1ull);
    nxt_item = it;
    if (it < nitems) {
      const uint32_t f = w.item_file[it];
      nxt_f = f;
      nxt_fd = w.fd[f];
      nxt_size = w.size[f];
      nxt_base = w.item_base[f];
    }
  };
  for (uint32_t i = tid; i < kCountSlots; i += nthr) {  // dynamic smem is not cleared between launches
    S.ckey[i] = 0;
    S.ccnt[i] = 0;
  }
  if (tid == 0) prefetch();
  long long t_prev = clock64();
  auto lap = [&](int k) {
    if (w.prof && tid == 0) {
      const long long t = clock64();
      atomicAdd(&w.prof[k], (unsigned long long)(t - t_prev));
      t_prev = t;
    }
  };
  for (;;) {
    __syncthreads();
    lap(0);  // 0: waiting at the loop-top barrier (end of flush)
    const uint64_t item = nxt_item;
    if (item >= nitems) break;
    const uint32_t f = nxt_f;
    S.hf = splitmix64(f);
    const int fd = nxt_fd;
    const uint64_t size = nxt_size;
    const uint64_t s = (item - nxt_base) * chunk;
    if (tid == 0) {
      nocc_s = 0;
      spilled_s = 0;
    }
    const uint64_t e = min(size, s + chunk);
    const uint64_t ws = s >= kPre ? s - kPre : 0;
    const uint64_t we = min(size, e + kHalo);
    // file byte p lands at buf[kPre + p - s]; (dst - ws) % 16 == 0, so gread
    // moves the span with TMA (s is a multiple of the chunk, itself of 16)
    const uint32_t vlo = (uint32_t)(kPre - (s - ws)), vhi = vlo + (uint32_t)(we - ws);
    const int64_t r = gread(c, fd, ws, we - ws, S.buf + vlo);  // starts with a barrier
    lap(1);  // 1: gread
    if (r != (int64_t)(we - ws)) {
      if (tid == 0) {
        set_err(w, r < 0 ? r : -EIO);
        prefetch();
      }
      continue;
    }
    // pass 1: word-byte bits per 32-byte stripe; bytes outside [vlo, vhi) are non-word
    const uint32_t nstripe = (vhi + 31) / 32;
    for (uint32_t j = tid; j < nstripe; j += nthr)
      S.mask[j] = word_bits32(S.buf + 32 * j) & bit_range((int)vlo - 32 * (int)j, (int)vhi - 32 * (int)j);
    if (tid == 0) S.mask[nstripe] = 0;
    __syncthreads();
    lap(2);  // 2: pass 1
    if (tid == 0) prefetch();  // next item's fields, overlapping pass 2
    // pass 2, by rounds of 2 stripes per thread: the starts of tokens in
    // [s, e) = buf[kPre, kPre + e - s) are compacted into `tok`, then every
    // thread takes every nthr-th token (balanced whatever the text layout)
    const uint32_t olo = kPre, ohi = kPre + (uint32_t)(e - s);
    const uint32_t jlo = olo / 32, jhi = (ohi - 1) / 32;
    for (uint32_t r0 = jlo; r0 <= jhi; r0 += round_stripes) {
      uint32_t st[2];
      uint32_t cnt = 0;
#pragma unroll
      for (int q = 0; q < 2; ++q) {
        const uint32_t j = r0 + 2 * (uint32_t)tid + q;
        st[q] = 0;
        if (j <= jhi) {
          const uint32_t m = S.mask[j];
          const uint32_t prev = j ? S.mask[j - 1] >> 31 : 0u;
          st[q] = m & ~((m << 1) | prev) & bit_range((int)olo - 32 * (int)j, (int)ohi - 32 * (int)j);
        }
        cnt += __popc(st[q]);
      }
      uint32_t incl = cnt;
      for (int o = 1; o < 32; o <<= 1) {
        const uint32_t t = __shfl_up_sync(0xFFFFFFFFu, incl, o);
        if (lane >= o) incl += t;
      }
      if (lane == 31) warp_tot[wid] = incl;
      __syncthreads();
      uint32_t off = incl - cnt, total = 0;
      for (int q = 0; q < (nthr >> 5); ++q) {
        const uint32_t t = warp_tot[q];
        off += q < wid ? t : 0u;
        total += t;
      }
#pragma unroll
      for (int q = 0; q < 2; ++q) {
        const uint32_t jb = 32 * (r0 + 2 * (uint32_t)tid + q);
        for (uint32_t x = st[q]; x; x &= x - 1) tok[off++] = (uint16_t)(jb + __ffs(x) - 1);
      }
      __syncthreads();
      lap(3);  // 3: token list
      for (uint32_t q = tid; q < total; q += nthr) {
        const uint32_t i = tok[q], j = i >> 5, b = i & 31;
        const uint64_t win = ((uint64_t)S.mask[j + 1] << 32) | S.mask[j];
        const uint32_t L = __ffsll(~(win >> b)) - 1;  // run of word bytes; >= 33 means too long
        if (L <= 32)                                   // no dictionary word is longer (R12)
          scan_token(w, S, &nocc_s, &spilled_s, f, i, L, s + i - kPre, hits, hit_cap, acc);
      }
      lap(4);  // 4: own tokens
      __syncthreads();  // tok and warp_tot are reused by the next round
      lap(5);  // 5: waiting for the block's other tokens
    }
    // flush: a whole-file item with no spill owns its records; otherwise merge
    const uint32_t nocc = nocc_s;
    const bool direct = s == 0 && e == size && !spilled_s && rec;
    if (direct && tid == 0 && nocc) rbase_s = atomicAdd(&w.vars[V_NREC], (unsigned long long)nocc);
    __syncthreads();
    if (w.prof && tid == 0) atomicAdd(&w.prof[7], 1ull);  // 7: items
    for (uint32_t q = tid; q < nocc; q += nthr) {
      const uint32_t cs = S.olist[q];
      const uint32_t k = S.ckey[cs] - 1, cnt = S.ccnt[cs];
      S.ckey[cs] = 0;
      S.ccnt[cs] = 0;
      if (direct) {
        atomicAdd((unsigned long long*)&totals[k], (unsigned long long)cnt);
        const uint64_t idx = rbase_s + q;
        if (idx < rec_cap) {
          rec[3 * idx] = f;
          rec[3 * idx + 1] = k;
          rec[3 * idx + 2] = cnt;
        } else {
          set_err(w, -ENOSPC);
        }
      } else {
        pair_add(w, f, k, cnt);
      }
    }
  }
  // block-level digest reduction
  for (int o = 16; o; o >>= 1) {
    acc.dsum += __shfl_xor_sync(0xFFFFFFFFu, acc.dsum, o);
    acc.dxor ^= __shfl_xor_sync(0xFFFFFFFFu, acc.dxor, o);
    acc.nh += __shfl_xor_sync(0xFFFFFFFFu, acc.nh, o);
  }
  if (lane == 0) {
    atomicAdd(&w.vars[V_DSUM], (unsigned long long)acc.dsum);
    atomicXor(&w.vars[V_DXOR], (unsigned long long)acc.dxor);
    atomicAdd(&w.vars[V_NHITS], (unsigned long long)acc.nh);
  }
}

// ------------------------------------------------------------ warp-item scan
// The same method as k_grep_scan with one WARP per item (warp-collective
// gread_warp, the paper's design point P:L256-271): no block barrier in the
// item loop, so a warp waiting on its lookups or probes never holds up the
// others. Items are smaller (the chunk, e.g. 8 KiB) so a warp's buffer, mask,
// count table and token list fit in ~16 KiB of shared memory.
constexpr uint32_t kWarpSlots = 256;  // per-warp count table (overflow spills to the global table)
constexpr uint32_t kWarpTok = 2048;   // bytes: 64 stripes x <= 16 token starts x u16

__host__ __device__ __forceinline__ uint32_t warp_region_bytes(uint32_t chunk) {
  const uint32_t buf_bytes = (kPre + chunk + kHalo + kSlack + 15) & ~15u;
  const uint32_t nstripe_max = (kPre + chunk + kHalo + 31) / 32;
  return buf_bytes + ((nstripe_max + 1 + 3) & ~3u) * 4 + kWarpSlots * 8 + kWarpSlots * 2 + kWarpTok + 16;
}

__global__ void __launch_bounds__(256) k_grep_scan_warp(const gfs_ctx* c, GrepWork w, uint32_t chunk,
                                                         uint64_t* hits, uint64_t hit_cap, uint64_t* totals,
                                                         uint32_t* rec, uint64_t rec_cap) {
  extern __shared__ __align__(16) uint8_t sm[];
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
  uint8_t* base = sm + (size_t)wid * warp_region_bytes(chunk);
  const uint32_t buf_bytes = (kPre + chunk + kHalo + kSlack + 15) & ~15u;
  const uint32_t nstripe_max = (kPre + chunk + kHalo + 31) / 32;
  ScanSmem S;
  S.buf = base;
  S.mask = (uint32_t*)(base + buf_bytes);
  S.ckey = S.mask + ((nstripe_max + 1 + 3) & ~3u);
  S.ccnt = S.ckey + kWarpSlots;
  S.olist = (uint16_t*)(S.ccnt + kWarpSlots);
  S.cmask = kWarpSlots - 1;
  uint16_t* tok = S.olist + kWarpSlots;
  uint32_t* wv = (uint32_t*)((uint8_t*)tok + kWarpTok);  // [0] occupied slots, [1] spilled
  const uint64_t nitems = w.vars[V_NITEMS];
  ScanAcc acc{0, 0, 0};
  for (uint32_t i = lane; i < kWarpSlots; i += 32) {  // dynamic smem is not cleared between launches
    S.ckey[i] = 0;
    S.ccnt[i] = 0;
  }
  // lane 0 claims the next item; its fields are loaded by every lane (broadcast)
  uint64_t item = 0;
  if (lane == 0) item = atomicAdd(&w.vars[V_NEXT], 1ull);
  item = __shfl_sync(0xFFFFFFFFu, item, 0);
  while (item < nitems) {
    const uint32_t f = w.item_file[item];
    const int fd = w.fd[f];
    const uint64_t size = w.size[f];
    const uint64_t s = (item - w.item_base[f]) * chunk;
    uint64_t next = 0;  // claimed now, so its fields' loads overlap this item
    if (lane == 0) {
      next = atomicAdd(&w.vars[V_NEXT], 1ull);
      wv[0] = 0;
      wv[1] = 0;
    }
    S.hf = splitmix64(f);
    const uint64_t e = min(size, s + chunk);
    const uint64_t ws = s >= kPre ? s - kPre : 0;
    const uint64_t we = min(size, e + kHalo);
    const uint32_t vlo = (uint32_t)(kPre - (s - ws)), vhi = vlo + (uint32_t)(we - ws);
    const int64_t r = gread_warp(c, fd, ws, we - ws, S.buf + vlo);
    next = __shfl_sync(0xFFFFFFFFu, next, 0);
    if (r != (int64_t)(we - ws)) {
      if (lane == 0) set_err(w, r < 0 ? r : -EIO);
      item = next;
      continue;
    }
    // pass 1: word-byte bits per 32-byte stripe; bytes outside [vlo, vhi) are non-word
    const uint32_t nstripe = (vhi + 31) / 32;
    for (uint32_t j = lane; j < nstripe; j += 32)
      S.mask[j] = word_bits32(S.buf + 32 * j) & bit_range((int)vlo - 32 * (int)j, (int)vhi - 32 * (int)j);
    if (lane == 0) S.mask[nstripe] = 0;
    __syncwarp();
    // pass 2, 64 stripes per round: token starts in [s, e) compacted into tok
    const uint32_t olo = kPre, ohi = kPre + (uint32_t)(e - s);
    const uint32_t jlo = olo / 32, jhi = (ohi - 1) / 32;
    for (uint32_t r0 = jlo; r0 <= jhi; r0 += 64) {
      uint32_t st[2];
      uint32_t cnt = 0;
#pragma unroll
      for (int q = 0; q < 2; ++q) {
        const uint32_t j = r0 + 2 * (uint32_t)lane + q;
        st[q] = 0;
        if (j <= jhi) {
          const uint32_t m = S.mask[j];
          const uint32_t prev = j ? S.mask[j - 1] >> 31 : 0u;
          st[q] = m & ~((m << 1) | prev) & bit_range((int)olo - 32 * (int)j, (int)ohi - 32 * (int)j);
        }
        cnt += __popc(st[q]);
      }
      uint32_t incl = cnt;
      for (int o = 1; o < 32; o <<= 1) {
        const uint32_t t = __shfl_up_sync(0xFFFFFFFFu, incl, o);
        if (lane >= o) incl += t;
      }
      const uint32_t total = __shfl_sync(0xFFFFFFFFu, incl, 31);
      uint32_t off = incl - cnt;
#pragma unroll
      for (int q = 0; q < 2; ++q) {
        const uint32_t jb = 32 * (r0 + 2 * (uint32_t)lane + q);
        for (uint32_t x = st[q]; x; x &= x - 1) tok[off++] = (uint16_t)(jb + __ffs(x) - 1);
      }
      __syncwarp();
      for (uint32_t q = lane; q < total; q += 32) {
        const uint32_t i = tok[q], j = i >> 5, b = i & 31;
        const uint64_t win = ((uint64_t)S.mask[j + 1] << 32) | S.mask[j];
        const uint32_t L = __ffsll(~(win >> b)) - 1;  // run of word bytes; >= 33 means too long
        if (L <= 32)                                   // no dictionary word is longer (R12)
          scan_token(w, S, &wv[0], &wv[1], f, i, L, s + i - kPre, hits, hit_cap, acc);
      }
      __syncwarp();  // tok is reused by the next round
    }
    // flush: a whole-file item with no spill owns its records; otherwise merge
    const uint32_t nocc = wv[0];
    const bool direct = s == 0 && e == size && !wv[1] && rec;
    unsigned long long rbase = 0;
    if (direct && lane == 0 && nocc) rbase = atomicAdd(&w.vars[V_NREC], (unsigned long long)nocc);
    rbase = __shfl_sync(0xFFFFFFFFu, rbase, 0);
    for (uint32_t q = lane; q < nocc; q += 32) {
      const uint32_t cs = S.olist[q];
      const uint32_t k = S.ckey[cs] - 1, cnt = S.ccnt[cs];
      S.ckey[cs] = 0;
      S.ccnt[cs] = 0;
      if (direct) {
        atomicAdd((unsigned long long*)&totals[k], (unsigned long long)cnt);
        const uint64_t idx = rbase + q;
        if (idx < rec_cap) {
          rec[3 * idx] = f;
          rec[3 * idx + 1] = k;
          rec[3 * idx + 2] = cnt;
        } else {
          set_err(w, -ENOSPC);
        }
      } else {
        pair_add(w, f, k, cnt);
      }
    }
    __syncwarp();  // count table and wv are reset before the next item uses them
    item = next;
  }
  for (int o = 16; o; o >>= 1) {
    acc.dsum += __shfl_xor_sync(0xFFFFFFFFu, acc.dsum, o);
    acc.dxor ^= __shfl_xor_sync(0xFFFFFFFFu, acc.dxor, o);
    acc.nh += __shfl_xor_sync(0xFFFFFFFFu, acc.nh, o);
  }
  if (lane == 0) {
    atomicAdd(&w.vars[V_DSUM], (unsigned long long)acc.dsum);
    atomicXor(&w.vars[V_DXOR], (unsigned long long)acc.dxor);
    atomicAdd(&w.vars[V_NHITS], (unsigned long long)acc.nh);
  }
}

__global__ void k_grep_close(const gfs_ctx* c, GrepWork w) {
  const uint32_t nfiles = (uint32_t)w.vars[V_NFILES];
  for (uint32_t f = blockIdx.x; f < nfiles; f += gridDim.x) {
    const int fd = w.fd[f];
    if (fd >= 0) gclose(c, fd);
  }
}

// Unique records from the (file, word) table + word totals. A block takes
// 1024 consecutive slots (4 per thread, 64 contiguous bytes), scans the valid
// counts and reserves its output range with one atomic.
__global__ void __launch_bounds__(256) k_grep_compact(GrepWork w, uint32_t* rec, uint64_t rec_cap,
                                                      uint64_t* totals) {
  __shared__ uint32_t warp_tot[8];
  __shared__ unsigned long long base_s;
  const int tid = threadIdx.x, lane = tid & 31, wid = tid >> 5;
  const uint64_t n = w.pair_mask + 1;  // a power of two >= 1024
  for (uint64_t blk = blockIdx.x; blk * 1024 < n; blk += gridDim.x) {
    const uint64_t i0 = blk * 1024 + (uint64_t)tid * 4;
    const uint4* src = (const uint4*)(w.pair + 2 * i0);
    uint64_t key[4], cnt[4];
    uint32_t nv = 0;
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      const uint4 v = src[q];
      key[q] = ((uint64_t)v.y << 32) | v.x;
      cnt[q] = ((uint64_t)v.w << 32) | v.z;
      nv += key[q] != kPairEmpty;
    }
    uint32_t incl = nv;  // inclusive scan in the warp, then across warps
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t t = __shfl_up_sync(0xFFFFFFFFu, incl, o);
      if (lane >= o) incl += t;
    }
    if (lane == 31) warp_tot[wid] = incl;
    __syncthreads();
    uint32_t before = 0, all = 0;
    for (int q = 0; q < 8; ++q) {
      const uint32_t t = warp_tot[q];
      before += q < wid ? t : 0u;
      all += t;
    }
    if (tid == 0) base_s = all ? atomicAdd(&w.vars[V_NREC], (unsigned long long)all) : 0ull;
    __syncthreads();
    uint64_t idx = base_s + before + incl - nv;
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      if (key[q] == kPairEmpty) continue;
      const uint32_t k = (uint32_t)key[q];
      atomicAdd((unsigned long long*)&totals[k], (unsigned long long)cnt[q]);
      if (idx < rec_cap) {
        rec[3 * idx] = (uint32_t)(key[q] >> 32);
        rec[3 * idx + 1] = k;
        rec[3 * idx + 2] = (uint32_t)cnt[q];
      } else if (rec) {
        set_err(w, -ENOSPC);
      }
      ++idx;
    }
    __syncthreads();  // warp_tot / base_s reuse
  }
}

__global__ void k_grep_init(GrepWork w, uint32_t max_words) {
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  const uint64_t t = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x;
  for (uint64_t i = t; i <= w.pair_mask; i += stride) {
    w.pair[2 * i] = kPairEmpty;
    w.pair[2 * i + 1] = 0;
  }
  for (uint64_t i = t; i <= w.table_mask; i += stride) w.table[i] = 0;
  for (uint64_t i = t; i < max_words; i += stride) {
    w.dup_head[i] = 0;
    w.dup_next[i] = 0;
  }
  if (t < V_NVARS) w.vars[t] = 0;
}

__global__ void k_grep_summary(GrepWork w, uint64_t* out) {
  if (threadIdx.x == 0) {
    out[0] = w.vars[V_NREC];
    out[1] = w.vars[V_NHITS];
    out[2] = w.vars[V_DSUM];
    out[3] = w.vars[V_DXOR];
    out[4] = w.vars[V_NFILES];
    out[5] = w.vars[V_NWORDS];
    out[6] = w.vars[V_BYTES];
    out[7] = w.vars[V_ERR];
    out[8] = w.vars[V_NLISTED];
    out[9] = w.vars[V_NITEMS];
  }
}

uint64_t pow2_at_least(uint64_t x) {
  uint64_t p = 1;
  while (p < x) p <<= 1;
  return p;
}

struct Layout {
  uint64_t off[16];
  uint64_t total;
  uint64_t max_items;
};

Layout layout(const gfs_grep_params* p) {
  Layout L{};
  const uint64_t tcap = pow2_at_least(p->max_words * 8ull < 1024 ? 1024 : p->max_words * 8ull);
  const uint64_t pcap = pow2_at_least(p->pair_cap < 1024 ? 1024 : p->pair_cap);
  // items: one per chunk of corpus plus one partial chunk per file
  L.max_items = p->corpus_cap / (p->chunk ? p->chunk : 1) + p->max_files + 1;
  const uint64_t sizes[] = {
      (uint64_t)p->max_words * 32,                         // dict
      tcap * 8,                                            // table
      (uint64_t)p->max_words * 4,                          // dup_head
      (uint64_t)p->max_words * 4,                          // dup_next
      p->list_cap + 64,                                    // list
      (p->list_cap / kListChunk + 2) * 4,                  // list_chunk
      (uint64_t)p->max_files * kMaxPath,                   // paths
      (uint64_t)p->max_files * 4,                          // fd
      (uint64_t)p->max_files * 8,                          // size
      ((uint64_t)p->max_files + 1) * 8,                    // item_base
      L.max_items * 4,                                     // item_file
      pcap * 16,                                           // pair
      0,                                                   // (unused)
      V_NVARS * 8,                                         // vars
  };
  uint64_t o = 0;
  for (int i = 0; i < 14; ++i) {
    L.off[i] = o;
    o += (sizes[i] + 255) & ~255ull;
  }
  L.total = o;
  return L;
}

uint32_t scan_smem(uint32_t chunk, uint32_t block) {
  const uint32_t buf_bytes = (kPre + chunk + kHalo + kSlack + 15) & ~15u;
  const uint32_t nstripe_max = (kPre + chunk + kHalo + 31) / 32;
  return buf_bytes + ((nstripe_max + 1 + 3) & ~3u) * 4 + 2 * kCountSlots * 4 + kCountSlots * 2 +
         64 * block;  // token list: <= 32 starts per thread per round (2 bytes each)
}

}  // namespace

GFS_API uint64_t gfs_grep_work_bytes(const gfs_grep_params* p) { return p ? layout(p).total : 0; }

GFS_API int gfs_grep(gfs_handle* h, void* stream, const char* dict_path, const char* list_path,
                     const gfs_grep_params* p, void* d_work, uint32_t* d_rec, uint64_t rec_cap, uint64_t* d_totals,
                     uint64_t* d_hits, uint64_t* d_summary) {
  if (!h || !dict_path || !list_path || !p || !d_work || !d_totals || !d_summary || p->max_files == 0 ||
      p->max_words == 0 || p->max_words >= (1u << 26) || p->chunk == 0 || (p->chunk & 15) || p->chunk + kPre + kHalo > 65536 ||  // u16 token offsets
      p->grid == 0 || p->block == 0 || p->block > 256 || (p->block & 31))
    return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  const Layout L = layout(p);
  uint8_t* base = (uint8_t*)d_work;
  GrepWork w;
  w.dict = base + L.off[0];
  w.table = (uint64_t*)(base + L.off[1]);
  w.table_mask = (uint32_t)(pow2_at_least(p->max_words * 8ull < 1024 ? 1024 : p->max_words * 8ull) - 1);
  w.dup_head = (uint32_t*)(base + L.off[2]);
  w.dup_next = (uint32_t*)(base + L.off[3]);
  w.list = base + L.off[4];
  w.list_chunk = (uint32_t*)(base + L.off[5]);
  w.paths = (char*)(base + L.off[6]);
  w.fd = (int32_t*)(base + L.off[7]);
  w.size = (uint64_t*)(base + L.off[8]);
  w.item_base = (uint64_t*)(base + L.off[9]);
  w.item_file = (uint32_t*)(base + L.off[10]);
  w.max_items = L.max_items;
  w.pair = (uint64_t*)(base + L.off[11]);
  w.pair_mask = pow2_at_least(p->pair_cap < 1024 ? 1024 : p->pair_cap) - 1;
  w.vars = (unsigned long long*)(base + L.off[13]);

  // staged strings: dict path, list path, list directory
  static char* d_str = nullptr;
  static char* h_str = nullptr;
  static cudaEvent_t ev = nullptr;
  if (!d_str) {
    if (cudaMalloc((void**)&d_str, 3 * kMaxPath) != cudaSuccess) return -ENOMEM;
    if (cudaHostAlloc((void**)&h_str, 3 * kMaxPath, cudaHostAllocPortable) != cudaSuccess) return -ENOMEM;
    cudaEventCreateWithFlags(&ev, cudaEventDisableTiming);
  } else {
    cudaEventSynchronize(ev);
  }
  const size_t nd = strlen(dict_path), nl = strlen(list_path);
  if (nd >= kMaxPath || nl >= kMaxPath) return -ENAMETOOLONG;
  memcpy(h_str, dict_path, nd + 1);
  memcpy(h_str + kMaxPath, list_path, nl + 1);
  const char* slash = strrchr(list_path, '/');
  size_t dl = 0;
  if (slash) {
    dl = (size_t)(slash - list_path);
    memcpy(h_str + 2 * kMaxPath, list_path, dl);
  } else {
    h_str[2 * kMaxPath] = '.';
    dl = 1;
  }
  h_str[2 * kMaxPath + dl] = 0;
  cudaMemcpyAsync(d_str, h_str, 3 * kMaxPath, cudaMemcpyHostToDevice, s);
  cudaEventRecord(ev, s);

  const gfs_ctx* c = gfs_device_ctx(h);
  // GFS_GREP_WARP=1: one warp per item (k_grep_scan_warp)
  const bool warp_items = getenv("GFS_GREP_WARP") && *getenv("GFS_GREP_WARP") == '1';
  const uint32_t smem = warp_items ? warp_region_bytes(p->chunk) * (p->block / 32) : scan_smem(p->chunk, p->block);
  if (smem > 227 * 1024) return -EINVAL;
  if (warp_items && p->block / 32 > GFS_WARP_API_MAX_WARPS) return -EINVAL;
  cudaFuncSetAttribute(warp_items ? (const void*)k_grep_scan_warp : (const void*)k_grep_scan,
                       cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  // GFS_GREP_DEBUG=1: synchronise after each stage, print its time and the first error
  const bool dbg = getenv("GFS_GREP_DEBUG") && *getenv("GFS_GREP_DEBUG") == '1';
  static unsigned long long* d_prof = nullptr;
  w.prof = nullptr;
  if (getenv("GFS_GREP_PROF") && *getenv("GFS_GREP_PROF") == '1') {
    if (!d_prof && cudaMalloc((void**)&d_prof, 8 * sizeof(unsigned long long)) != cudaSuccess) d_prof = nullptr;
    if (d_prof) cudaMemsetAsync(d_prof, 0, 8 * sizeof(unsigned long long), s);
    w.prof = d_prof;
  }
  struct timespec ts_prev;
  clock_gettime(CLOCK_MONOTONIC, &ts_prev);
  auto stage = [&](const char* name) {
    if (!dbg) return;
    cudaError_t e = cudaStreamSynchronize(s);
    struct timespec ts;
    clock_gettime(CLOCK_MONOTONIC, &ts);
    unsigned long long v[V_NVARS];
    cudaMemcpy(v, w.vars, sizeof(v), cudaMemcpyDeviceToHost);
    fprintf(stderr, "gfs_grep[%s]: %.3f ms cuda=%s err=%lld nfiles=%llu nwords=%llu nitems=%llu bytes=%llu\n", name,
            (ts.tv_sec - ts_prev.tv_sec) * 1e3 + (ts.tv_nsec - ts_prev.tv_nsec) * 1e-6, cudaGetErrorString(e),
            (long long)v[V_ERR], v[V_NFILES], v[V_NWORDS], v[V_NITEMS], v[V_BYTES]);
    ts_prev = ts;
  };
  const uint64_t lb = p->list_cap / kListChunk + 1, lr = p->list_cap / kListRead + 1;
  const uint32_t list_blocks = (uint32_t)(lb < 1024 ? lb : 1024);
  // one opener per 64 KiB piece: a block that opens the list after all others
  // closed it would re-validate it with the host (close-to-open)
  const uint32_t read_blocks = (uint32_t)(lr < 1024 ? lr : 1024);
  k_grep_init<<<1024, 256, 0, s>>>(w, p->max_words);
  k_grep_hold<<<1, 32, 0, s>>>(c, d_str, d_str + kMaxPath, w, 0);
  k_grep_dict<<<64, 256, 0, s>>>(c, d_str, w, p->max_words);
  stage("dict");
  k_grep_list_read<<<read_blocks, 256, 0, s>>>(c, d_str + kMaxPath, w, p->list_cap);
  k_grep_list_count<<<list_blocks, 256, 0, s>>>(w);
  k_grep_list_scan<<<1, 32, 0, s>>>(w, p->max_files);
  k_grep_list_emit<<<list_blocks, 256, 0, s>>>(w, d_str + 2 * kMaxPath, (uint32_t)dl, p->max_files);
  stage("list");
  // gopen is block-collective with one leader thread: many one-warp blocks
  // keep more opens in flight (host RPCs when cold, L2 round trips when warm)
  int dev = 0, nsm = 148;
  cudaGetDevice(&dev);
  cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, dev);
  k_grep_open<<<nsm * 16, 32, 0, s>>>(c, w, p->chunk);
  stage("open");
  k_grep_plan<<<1, 1024, 0, s>>>(w);
  k_grep_items<<<256, 256, 0, s>>>(w);
  cudaMemsetAsync(d_totals, 0, (size_t)p->max_words * 8, s);
  // persistent scan grid: every resident block slot once (p->grid caps it)
  int occ = 1;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, warp_items ? (const void*)k_grep_scan_warp
                                                                 : (const void*)k_grep_scan, (int)p->block, smem);
  // GFS_GREP_BPS=n: at most n scan blocks per SM, the rest of the SM's
  // L1/shared-memory array left to L1 (dictionary buckets of frequent words)
  if (getenv("GFS_GREP_BPS")) {
    const int cap = atoi(getenv("GFS_GREP_BPS"));
    if (cap > 0 && cap < occ) occ = cap;
    const int pct = (int)((occ * (uint64_t)(smem + 1024) * 100 + 228 * 1024 - 1) / (228 * 1024));
    cudaFuncSetAttribute(k_grep_scan, cudaFuncAttributePreferredSharedMemoryCarveout, pct < 100 ? pct : 100);
  }
  const uint32_t scan_grid = (uint32_t)(occ > 0 ? occ : 1) * (uint32_t)nsm;
  if (warp_items)
    k_grep_scan_warp<<<scan_grid < p->grid ? scan_grid : p->grid, p->block, smem, s>>>(
        c, w, p->chunk, d_hits, d_hits ? p->hit_cap : 0, d_totals, d_rec, d_rec ? rec_cap : 0);
  else
    k_grep_scan<<<scan_grid < p->grid ? scan_grid : p->grid, p->block, smem, s>>>(
        c, w, p->chunk, d_hits, d_hits ? p->hit_cap : 0, d_totals, d_rec, d_rec ? rec_cap : 0);
  stage("scan");
  if (!p->keep_open) k_grep_close<<<nsm * 16, 32, 0, s>>>(c, w);
  k_grep_compact<<<nsm * 8, 256, 0, s>>>(w, d_rec, d_rec ? rec_cap : 0, d_totals);
  k_grep_hold<<<1, 32, 0, s>>>(c, d_str, d_str + kMaxPath, w, 1);
  k_grep_summary<<<1, 32, 0, s>>>(w, d_summary);
  stage("done");
  if (w.prof) {
    unsigned long long pv[8];
    cudaMemcpyAsync(pv, w.prof, sizeof(pv), cudaMemcpyDeviceToHost, s);
    cudaStreamSynchronize(s);
    const double tot = (double)(pv[0] + pv[1] + pv[2] + pv[3] + pv[4] + pv[5]) + 1e-9;
    fprintf(stderr, "gfs_grep[scan prof, thread 0 cycles]: items=%llu loop-top=%.1f%% gread=%.1f%% pass1=%.1f%% "
            "toklist=%.1f%% tokens=%.1f%% wait-others=%.1f%% (%.0f cycles/item)\n", pv[7], 100 * pv[0] / tot,
            100 * pv[1] / tot, 100 * pv[2] / tot, 100 * pv[3] / tot, 100 * pv[4] / tot, 100 * pv[5] / tot,
            tot / (double)(pv[7] ? pv[7] : 1));
  }
  const cudaError_t e = cudaGetLastError();
  if (e != cudaSuccess) fprintf(stderr, "gfs_grep: launch failed: %s\n", cudaGetErrorString(e));
  return e == cudaSuccess ? 0 : -EIO;
}
