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
//   k_grep_list_* gread the file list, find the line starts (parallel over the
//                 list), record each line's offset;
//   k_grep_open   one warp per file builds its path from the list line, gopen
//                 (the first gopen goes to the host), gfstat;
//   k_grep_items  one 32-byte descriptor per work item: a file of one chunk,
//                 a file of up to `whole_max` bytes scanned chunk after chunk
//                 by one block (these first, most chunks first), or one chunk
//                 of a larger file: one round trip per item;
//   k_grep_scan   persistent blocks pull items. gread brings the item plus a
//                 halo into shared memory (TMA). Pass 1 classifies 32-byte
//                 stripes into word-byte bit masks (SWAR, 4 bytes per op); pass
//                 2 gives each thread the tokens that start in its stripe:
//                 length from the masks, bytes gathered as 8 zero-padded words,
//                 one hash, one probe of the (L2-resident) table, an exact
//                 32-byte compare on a fingerprint match. Counts per item in
//                 shared memory; a whole-file item emits its (file, word,
//                 count) records directly (into a record page the block
//                 reserved), chunks of files above `whole_max` merge through
//                 a global (file, word) table;
//   k_grep_close  gclose every file (unless kept open for warm re-runs);
//   k_grep_compact emit the merged records and their word totals, and leave
//                 the (file, word) table empty for the next run;
//   k_grep_pack_* pack the record pages into the caller's contiguous array.
// Word bytes are [A-Za-z0-9_] (GNU grep -w under LC_ALL=C, R10).
#include <cuda_runtime.h>
#include <errno.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>

#include <string>

#include "gpufs.h"
#include "gpufs_device.cuh"
#include "gfs_launch.h"

#define GFS_API extern "C" __attribute__((visibility("default")))

using namespace gfs;

namespace {

constexpr uint32_t kMaxPath = GFS_MAX_PATH;
constexpr uint32_t kHalo = 48;      // bytes after a chunk: a token starting inside may run 33 bytes
constexpr uint32_t kPre = 16;       // bytes before a chunk (one needed for the boundary test)
constexpr uint32_t kSlack = 64;     // gathers read up to 48 bytes past a token start
constexpr uint32_t kListRead = 65536;  // list file gread granularity
constexpr uint32_t kListChunk = 4096;  // list parse granularity (one block per chunk)
constexpr uint64_t kPairEmpty = ~0ull;
constexpr uint64_t kDupBit = 1ull << 63;  // table entry: the word has duplicates
constexpr uint64_t kKeepMagic = 0x31504545504b5247ull;  // GRKPEEP1: the persistent words are initialised
constexpr uint64_t kPairsClean = 0x4e41454c43524150ull;  // PAIRCLEAN: the (file, word) table is empty
constexpr uint32_t kRecPage = 4096;  // records per output page (>= the count table: one item's records fit)
constexpr uint32_t kNoPage = 0xFFFFFFFFu;

// One work item (a whole file, or a chunk of a large one), precomputed by
// k_grep_items so the scan needs one round trip per item (32 bytes).
struct ItemDesc {
  uint64_t roff;    // file offset of the read: chunk start - pre
  uint32_t f;       // list index
  int32_t fd;
  uint32_t gid;     // reported file id
  uint32_t rlen;    // bytes to read (chunk + halos, clipped at EOF); a multi-chunk whole file: its size
  uint32_t body;    // bytes whose token starts this item counts (the chunk); multi-chunk: the chunk count
  uint32_t meta;    // bit 31: a whole file (records emitted directly); bit 30: multi-chunk whole file;
                    // bits 0..4: pre (bytes before the chunk)
};
constexpr uint32_t kMaxWholeChunks = 31;  // chunks of a file one block scans whole (histogram buckets)

struct GrepWork {
  // dictionary
  uint8_t* dict;          // max_words * 32
  uint64_t* table;        // (dup << 63) | (fp31 << 32) | (len << 26) | (k + 1); 0 = empty
  uint32_t table_mask;
  uint32_t* dup_head;     // per primary word: first duplicate + 1
  uint32_t* dup_next;     // per word: next duplicate + 1
  uint32_t* filt;         // one bit per filter_index() value of the words' hashes (L1-resident)
  uint32_t filt_log2;     // log2 of the filter's bits
  // file list
  uint8_t* list;          // list_cap bytes
  uint32_t* list_chunk;   // per list chunk: line starts (then exclusive prefix)
  uint64_t* line_off;     // per file: offset of its line in the list
  const uint32_t* file_ids;  // per file: the id used in records, hits and the digest (NULL: the list index)
  int32_t* fd;
  uint64_t* size;
  struct ItemDesc* desc;  // item -> what to read and where it goes (k_grep_items)
  uint64_t max_items;
  uint32_t chunk;         // item bytes
  uint32_t whole_chunks;  // a file of 2..whole_chunks chunks is one item, scanned whole by one block
  uint32_t cslots;        // count table slots per scan block (power of two)
  // (file, word) -> count table
  uint64_t* pair;         // slot i: pair[2i] = (file << 32) | word (or empty), pair[2i+1] = count
  uint64_t pair_mask;
  uint32_t* ptouch;       // one bit per 256 slots that hold (or held) a pair this run: compact skips the rest
  // output records, staged in pages: a block reserves a page of kRecPage
  // records with ONE atomic and fills it privately (a global counter bumped
  // per record or per warp serialises at one L2 address, ~14 ns each);
  // k_grep_pack then packs the used part of every page into d_rec
  uint32_t* rpool;        // pages of kRecPage records, 3 words each
  uint32_t* page_used;    // records in each reserved page
  uint64_t* page_base;    // exclusive prefix of page_used (k_grep_pack)
  uint64_t max_pages;
  // counters
  unsigned long long* vars;  // see V_*; cleared every run
  unsigned long long* keep;  // see K_*; persistent across runs (same work buffer)
  unsigned long long* prof;  // GFS_GREP_PROF=1: per-phase clock cycles of the scan's thread 0 (else null)
};
enum { V_NFILES = 0, V_NWORDS, V_NITEMS, V_NEXT, V_ERR, V_BYTES, V_NREC, V_NHITS, V_DSUM, V_DXOR, V_NLISTED,
       V_NEXTF, V_LISTSZ, V_HOLD_DICT, V_HOLD_LIST, V_NPAGES, V_PAIRS_DIRTY,
       V_NCHUNKED,                         // items of files split into chunks
       V_CUR_CHUNKED,                      // their placement cursor (k_grep_items)
       V_CUR_ONE,                          // one-chunk files: placement cursor = their count
       V_WHOLE_HIST,                       // [n]: multi-chunk whole files of n chunks
       V_WHOLE_CUR = V_WHOLE_HIST + kMaxWholeChunks + 1,  // [n]: their placement cursors
       V_NDIRECT = V_WHOLE_CUR + kMaxWholeChunks + 1,  // records the warp scan wrote straight into d_rec
       V_NVARS };
enum { K_MAGIC = 0, K_PAIRS, K_DICT_FD, K_LIST_FD, K_NKEEP };

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
  // 32-bit multiply-xorshift rounds (one IMAD each; a 64-bit multiply is ~4):
  // the low word picks the bucket, the high word is the 31-bit fingerprint
  uint32_t a = (w0 ^ (L * 0x9E3779B9u)) * 0x85EBCA6Bu;
  a ^= a >> 13;
  uint32_t b = (w1 + a) * 0xC2B2AE35u;
  b ^= b >> 16;
  a = (a ^ b) * 0x27D4EB2Fu;
  a ^= a >> 15;
  b = (b ^ (a >> 7)) * 0x165667B1u;
  b ^= b >> 15;
  return ((uint64_t)b << 32) | a;
}

// Low `nb` (0..4) bytes of a word.
__device__ __forceinline__ uint32_t low_bytes(uint32_t x, int nb) {
  return x & __funnelshift_lc(0xFFFFFFFFu, 0u, 8 * nb);
}

// Bytes [i, i + L) of buf (4-byte aligned shared memory, >= 36 readable
// bytes from i & ~3) as 8 zero-padded words: nine word loads and funnel
// shifts (no select chains).
__device__ __forceinline__ void token_words(const uint8_t* buf, uint32_t i, uint32_t L, uint32_t (&v)[8]) {
  const uint32_t* q = (const uint32_t*)(buf + (i & ~3u));
  const uint32_t r = (i & 3u) * 8;
  uint32_t wv[9];
#pragma unroll
  for (int j = 0; j < 9; ++j) wv[j] = q[j];
#pragma unroll
  for (int j = 0; j < 8; ++j) {
    const int nb = min(max((int)L - 4 * j, 0), 4);
    v[j] = __funnelshift_r(wv[j], wv[j + 1], r) & __funnelshift_lc(0xFFFFFFFFu, 0u, 8 * nb);
  }
}

// entry bits 32..62 hold a 31-bit fingerprint, 26..31 the length
__device__ __forceinline__ uint64_t entry_key(uint64_t h, uint32_t len) {
  return (((h >> 32) & 0x7FFFFFFFull) << 32) | ((uint64_t)len << 26);
}
__device__ __forceinline__ uint64_t key_bits(uint64_t e) { return (e & ~kDupBit) >> 26; }

// Pre-filter: a token whose hash has no dictionary word's bit set is not a
// word (no false negatives; ~1 in 5 non-words pass at 4.5 bits per word). The
// bitmap (<= 32 KiB) is read with an L1 evict_last hint: it stays in L1, so
// most non-words end without an L2 round trip.
__device__ __forceinline__ uint32_t filter_index(uint64_t h, uint32_t log2) {
  return (((uint32_t)(h >> 32) ^ (uint32_t)h) * 0x9E3779B1u) >> (32 - log2);
}
__device__ __forceinline__ uint32_t ld_filter(const uint32_t* p) {
  uint32_t v;
  asm("ld.global.nc.L1::evict_last.u32 %0, [%1];" : "=r"(v) : "l"(p));
  return v;
}

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

__device__ __forceinline__ void set_err(const GrepWork& w, long long e) { atomicMin((long long*)&w.vars[V_ERR], e); }

__device__ __forceinline__ uint32_t gid_of(const GrepWork& w, uint32_t f) { return w.file_ids ? w.file_ids[f] : f; }

// --------------------------------------------------------------- hold
// One block opens the dictionary and the list before the blocks that read
// them, and releases them after the run: the many short gopen/gclose pairs of
// the reading blocks then never drop the count to zero, which would make the
// next opener re-validate the file with the host (close-to-open).
// With keep_open the two stay open until the next run (which opens them
// again, then drops the previous run's references), like the corpus files.
__global__ void k_grep_hold(const __grid_constant__ gfs_ctx cv_, const char* dict_path, const char* list_path, const __grid_constant__ GrepWork w, int release,
                            int keep_open) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  if (!release) {
    const int a = gopen(c, dict_path, GFS_O_RDONLY);
    const int b = gopen(c, list_path, GFS_O_RDONLY);
    if (threadIdx.x == 0) {
      w.vars[V_HOLD_DICT] = (unsigned long long)(long long)a;
      w.vars[V_HOLD_LIST] = (unsigned long long)(long long)b;
      if (w.keep[K_MAGIC] != kKeepMagic) {  // first run on this work buffer
        w.keep[K_PAIRS] = 0;
        w.keep[K_DICT_FD] = (unsigned long long)-1ll;
        w.keep[K_LIST_FD] = (unsigned long long)-1ll;
        w.keep[K_MAGIC] = kKeepMagic;
      }
      w.vars[V_PAIRS_DIRTY] = w.keep[K_PAIRS] != kPairsClean;
      w.keep[K_PAIRS] = 0;  // dirty until this run's compact has emptied it again
    }
  } else {
    const int a = (int)(long long)w.vars[V_HOLD_DICT], b = (int)(long long)w.vars[V_HOLD_LIST];
    int ra = a, rb = b;  // references to drop now
    if (keep_open) {
      ra = (int)(long long)w.keep[K_DICT_FD];
      rb = (int)(long long)w.keep[K_LIST_FD];
    }
    if (ra >= 0) gclose(c, ra);
    if (rb >= 0) gclose(c, rb);
    if (threadIdx.x == 0) {
      w.keep[K_DICT_FD] = keep_open ? (unsigned long long)(long long)a : (unsigned long long)-1ll;
      w.keep[K_LIST_FD] = keep_open ? (unsigned long long)(long long)b : (unsigned long long)-1ll;
    }
  }
}

// --------------------------------------------------------------- init
__global__ void k_grep_init(const __grid_constant__ GrepWork w, uint32_t max_words) {
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  const uint64_t t = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x;
  for (uint64_t i = t; i <= w.table_mask; i += stride) w.table[i] = 0;
  for (uint64_t i = t; i < (1ull << w.filt_log2) / 32; i += stride) w.filt[i] = 0;
  for (uint64_t i = t; i < max_words; i += stride) {
    w.dup_head[i] = 0;
    w.dup_next[i] = 0;
  }
  if (t < V_NVARS) w.vars[t] = 0;
}

__host__ __device__ __forceinline__ uint64_t ptouch_words(uint64_t slots) { return (slots / 256 + 31) / 32; }

// The (file, word) table is emptied by every successful run's compact; only
// a fresh work buffer or a failed run leaves it dirty.
__global__ void k_grep_pairclear(const __grid_constant__ GrepWork w) {
  if (!w.vars[V_PAIRS_DIRTY]) return;
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i <= w.pair_mask; i += stride) {
    w.pair[2 * i] = kPairEmpty;
    w.pair[2 * i + 1] = 0;
  }
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < ptouch_words(w.pair_mask + 1); i += stride)
    w.ptouch[i] = 0;
}

// --------------------------------------------------------------- dictionary
__global__ void k_grep_dict(const __grid_constant__ gfs_ctx cv_, const char* dict_path, const __grid_constant__ GrepWork w, uint32_t max_words) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
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
        uint4 q0 = *(const uint4*)s, q1 = *(const uint4*)(s + 16);
        uint8_t b[32];
        memcpy(b, &q0, 16);
        memcpy(b + 16, &q1, 16);
        uint32_t n = 0;
        while (n < 32 && b[n]) ++n;
        bool ok = n > 0;
        for (uint32_t i = 0; i < n; ++i) ok &= is_word(b[i]);
        if (!ok) {  // empty slot or non-word byte (R13)
          set_err(w, -EINVAL);
          continue;
        }
        // zero the bytes after the word: the slot becomes the word's padded form
        for (uint32_t i = n; i < 32; ++i) b[i] = 0;
        memcpy(&q0, b, 16);
        memcpy(&q1, b + 16, 16);
        *(uint4*)s = q0;
        *(uint4*)(s + 16) = q1;
        const uint64_t h = tok_hash(q0.x, q0.y, n);
        const uint64_t ent = entry_key(h, n) | (k + 1);
        const uint32_t fi = filter_index(h, w.filt_log2);
        atomicOr(&w.filt[fi >> 5], 1u << (fi & 31));
        // linear probing from the start of the hash's 4-entry (32-byte) bucket:
        // lookups read a whole bucket per step (probe_bucket)
        uint32_t slot = (uint32_t)h & w.table_mask & ~3u;
        for (uint32_t probe = 0; probe <= w.table_mask; ++probe, slot = (slot + 1) & w.table_mask) {
          unsigned long long cur = atomicCAS((unsigned long long*)&w.table[slot], 0ull, (unsigned long long)ent);
          if (cur == 0) break;
          if (key_bits(cur) == key_bits(ent)) {  // same fingerprint and length: same word?
            const uint32_t kp = (uint32_t)(cur & ((1u << 26) - 1)) - 1;
            const uint8_t* t = w.dict + (size_t)kp * 32;
            bool same = true;
            for (uint32_t i = 0; i < n; ++i) same &= t[i] == b[i];
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
__global__ void k_grep_list_read(const __grid_constant__ gfs_ctx cv_, const char* list_path, const __grid_constant__ GrepWork w, uint64_t list_cap) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
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
__global__ void k_grep_list_count(const __grid_constant__ GrepWork w) {
  const uint64_t size = w.vars[V_LISTSZ];
  const uint64_t nch = (size + kListChunk - 1) / kListChunk;
  for (uint64_t ch = blockIdx.x; ch < nch; ch += gridDim.x) {
    const uint64_t a = ch * kListChunk, b = min(size, a + kListChunk);
    uint32_t n = 0;
    for (uint64_t i = a + threadIdx.x; i < b; i += blockDim.x) n += line_start(w.list, i);
    const uint32_t tot = __reduce_add_sync(0xFFFFFFFFu, n);
    __shared__ uint32_t wsum[32];
    if ((threadIdx.x & 31) == 0) wsum[threadIdx.x >> 5] = tot;
    __syncthreads();
    if (threadIdx.x == 0) {
      uint32_t t = 0;
      for (uint32_t q = 0; q < (blockDim.x + 31) / 32; ++q) t += wsum[q];
      w.list_chunk[ch] = t;
    }
    __syncthreads();
  }
}

// Pass 3 (one block): exclusive scan of the chunk counts.
__global__ void k_grep_list_scan(const __grid_constant__ GrepWork w, uint32_t max_files) {
  __shared__ uint32_t part[1024];
  const uint64_t size = w.vars[V_LISTSZ];
  const uint32_t nch = (uint32_t)((size + kListChunk - 1) / kListChunk);
  const uint32_t tid = threadIdx.x, nthr = blockDim.x;
  const uint32_t per = (nch + nthr - 1) / nthr;
  const uint32_t a = min(nch, tid * per), b = min(nch, a + per);
  uint32_t s = 0;
  for (uint32_t i = a; i < b; ++i) s += w.list_chunk[i];
  part[tid] = s;
  __syncthreads();
  if (tid == 0) {
    uint32_t run = 0;
    for (uint32_t q = 0; q < nthr; ++q) {
      const uint32_t v = part[q];
      part[q] = run;
      run += v;
    }
    if (run > max_files) set_err(w, -ENOSPC);
    w.vars[V_NFILES] = run < max_files ? run : max_files;
  }
  __syncthreads();
  uint32_t run = part[tid];
  for (uint32_t i = a; i < b; ++i) {
    const uint32_t v = w.list_chunk[i];
    w.list_chunk[i] = run;
    run += v;
  }
}

// Pass 4: the offset of every line (file index = rank among non-empty lines).
__global__ void k_grep_list_emit(const __grid_constant__ GrepWork w, uint32_t max_files) {
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
      if (start && k < max_files) w.line_off[k] = i;
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
// One warp per file: the path is the list line (relative lines are resolved
// against the list's directory, R15), assembled in shared memory,
// then gopen + gfstat. Counts the file's items: the histogram of multi-chunk
// whole files by chunk count, the chunks of larger files.
__device__ __forceinline__ uint64_t item_count(uint64_t size, uint32_t chunk) { return (size + chunk - 1) / chunk; }
__device__ __forceinline__ bool whole_multi(const GrepWork& w, uint64_t nch) { return nch >= 2 && nch <= w.whole_chunks; }
__global__ void __launch_bounds__(32) k_grep_open(const __grid_constant__ gfs_ctx cv_, const __grid_constant__ GrepWork w, const char* dir, uint32_t dir_len,
                                                  uint32_t max_files) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  __shared__ __align__(16) char pbuf[kMaxPath + 32];
  __shared__ uint32_t f_s;
  const int lane = threadIdx.x;
  const uint32_t nfiles = (uint32_t)w.vars[V_NFILES];
  const uint64_t lsize = w.vars[V_LISTSZ];
  for (;;) {
    if (lane == 0) f_s = (uint32_t)atomicAdd(&w.vars[V_NEXTF], 1ull);
    __syncwarp();
    const uint32_t f = f_s;
    if (f >= nfiles) break;
    // assemble the path: [dir '/'] line
    const uint64_t lo = w.line_off[f];
    const bool rel = w.list[lo] != '/';
    uint32_t o = 0;
    if (rel) {
      for (uint32_t q = lane; q < dir_len; q += 32) pbuf[q] = dir[q];
      if (lane == 0) pbuf[dir_len] = '/';
      o = dir_len + 1;
    }
    uint32_t n = 0;  // line length
    bool toolong = false;
    for (uint64_t base = lo;; base += 32) {
      const uint64_t i = base + lane;
      const uint8_t ch = i < lsize ? w.list[i] : (uint8_t)'\n';
      const uint32_t nl = __ballot_sync(0xFFFFFFFFu, ch == '\n');
      const uint32_t lim = nl ? (uint32_t)(__ffs(nl) - 1) : 32u;
      const uint32_t pos = o + (uint32_t)(base - lo) + lane;
      if ((uint32_t)lane < lim && pos < kMaxPath) pbuf[pos] = (char)ch;
      if (nl) {
        n = (uint32_t)(base - lo) + lim;
        break;
      }
      if (o + (uint32_t)(base - lo) + 32 >= kMaxPath) {
        toolong = true;
        break;
      }
    }
    if (o + n >= kMaxPath) toolong = true;
    if (lane == 0 && !toolong) pbuf[o + n] = 0;
    __syncwarp();
    int fd = -ENAMETOOLONG;
    if (!toolong) fd = gopen(c, pbuf, GFS_O_RDONLY | GFS_O_PREFETCH);  // first gopen: page 0 with the reply
    else if (lane == 0) set_err(w, -ENAMETOOLONG);
    const int64_t sz = fd >= 0 ? gfstat_size(c, fd) : fd;
    if (lane == 0) {
      w.fd[f] = fd;
      if (sz < 0) {
        set_err(w, sz);
        w.size[f] = 0;
      } else {
        w.size[f] = (uint64_t)sz;
        const uint64_t nch = item_count((uint64_t)sz, w.chunk);
        if (whole_multi(w, nch)) atomicAdd(&w.vars[V_WHOLE_HIST + nch], 1ull);
        else if (nch > 1) atomicAdd(&w.vars[V_NCHUNKED], (unsigned long long)nch);
        atomicAdd(&w.vars[V_BYTES], (unsigned long long)sz);
      }
    }
    __syncwarp();
  }
}

// --------------------------------------------------------------- items
// Item order: the multi-chunk whole files first, most chunks first (the
// longest items start first: no block is left with a long item at the end),
// then the chunks of larger files, then the one-chunk files. Positions come
// from cursors: per chunk count for the whole files (one atomic per group of
// equal counts in a warp), one per block for the rest (block scan). Order
// within a class is arbitrary; the results do not depend on it.
__global__ void __launch_bounds__(256) k_grep_items(const __grid_constant__ GrepWork w) {
  __shared__ unsigned long long base_s[kMaxWholeChunks + 2];  // [n]: first item of n-chunk whole files
  __shared__ unsigned long long blk_s[2];
  __shared__ uint32_t wsum[2][8];
  const int tid = threadIdx.x, lane = tid & 31, wid = tid >> 5;
  const uint32_t n = (uint32_t)w.vars[V_NFILES];
  if (tid == 0) {
    unsigned long long o = 0;
    for (uint32_t k = kMaxWholeChunks; k >= 2; --k) {
      base_s[k] = o;
      o += w.vars[V_WHOLE_HIST + k];
    }
    base_s[kMaxWholeChunks + 1] = o;  // = whole multi-chunk items; chunked items follow
    blk_s[0] = o;
    blk_s[1] = o + w.vars[V_NCHUNKED];  // one-chunk files follow the chunked ones
  }
  __syncthreads();
  const unsigned long long nwhole = blk_s[0], chunk_end = blk_s[1];
  for (uint32_t f0 = blockIdx.x * 256u; f0 < n; f0 += gridDim.x * 256u) {
    const uint32_t f = f0 + tid;
    const bool valid = f < n;
    const uint64_t size = valid ? w.size[f] : 0;
    const uint64_t nch = item_count(size, w.chunk);
    const bool multi = valid && whole_multi(w, nch);
    const uint32_t u_chunks = (valid && !multi && nch > 1) ? (uint32_t)nch : 0u;
    const uint32_t u_one = (valid && nch == 1) ? 1u : 0u;
    // block scan of both counts
    uint32_t a = u_chunks, b = u_one;
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t ta = __shfl_up_sync(0xFFFFFFFFu, a, o), tb = __shfl_up_sync(0xFFFFFFFFu, b, o);
      if (lane >= o) {
        a += ta;
        b += tb;
      }
    }
    if (lane == 31) {
      wsum[0][wid] = a;
      wsum[1][wid] = b;
    }
    __syncthreads();
    uint32_t oa = a - u_chunks, ob = b - u_one, ta = 0, tb = 0;
    for (int q = 0; q < 8; ++q) {
      oa += q < wid ? wsum[0][q] : 0u;
      ob += q < wid ? wsum[1][q] : 0u;
      ta += wsum[0][q];
      tb += wsum[1][q];
    }
    if (tid == 0) {
      blk_s[0] = ta ? atomicAdd(&w.vars[V_CUR_CHUNKED], (unsigned long long)ta) : 0;
      blk_s[1] = tb ? atomicAdd(&w.vars[V_CUR_ONE], (unsigned long long)tb) : 0;
    }
    // whole multi-chunk files: one atomic per group of equal chunk counts
    const uint32_t key = multi ? (uint32_t)nch : 0xFFFFFFFFu;
    const uint32_t peers = __match_any_sync(0xFFFFFFFFu, key);
    unsigned long long wpos = 0;
    if (multi) {
      const int leader = __ffs(peers) - 1;
      unsigned long long b0 = 0;
      if (lane == leader) b0 = atomicAdd(&w.vars[V_WHOLE_CUR + nch], (unsigned long long)__popc(peers));
      b0 = __shfl_sync(peers, b0, leader);
      wpos = base_s[nch] + b0 + __popc(peers & ((1u << lane) - 1u));
    }
    __syncthreads();
    if (valid && nch) {
      ItemDesc d;
      d.f = f;
      d.fd = w.fd[f];
      d.gid = gid_of(w, f);
      if (nch == 1 || multi) {  // a whole file
        d.roff = 0;
        d.rlen = (uint32_t)size;
        d.body = multi ? (uint32_t)nch : (uint32_t)size;
        d.meta = multi ? (3u << 30) : (1u << 31);
        const unsigned long long pos = multi ? wpos : chunk_end + blk_s[1] + ob;
        if (pos < w.max_items) w.desc[pos] = d;
      } else {  // chunk [s, e) with up to kPre bytes before and kHalo after
        const unsigned long long p0 = nwhole + blk_s[0] + oa;
        for (uint64_t i = 0; i < nch; ++i) {
          const uint64_t s = i * w.chunk, e = min(size, s + w.chunk);
          const uint64_t ws = s >= kPre ? s - kPre : 0, we = min(size, e + kHalo);
          d.roff = ws;
          d.rlen = (uint32_t)(we - ws);
          d.body = (uint32_t)(e - s);
          d.meta = (uint32_t)(s - ws);
          if (p0 + i < w.max_items) w.desc[p0 + i] = d;
        }
      }
    }
    __syncthreads();  // blk_s and wsum are reused
  }
}

// The item count (all classes, after k_grep_items) and its bound.
__device__ uint64_t count_items(const GrepWork& w) {
  unsigned long long t = w.vars[V_NCHUNKED] + w.vars[V_CUR_ONE];
  for (uint32_t k = 2; k <= kMaxWholeChunks; ++k) t += w.vars[V_WHOLE_HIST + k];
  return t;
}

// --------------------------------------------------------------- scan
// Bits [lo, hi) of a 32-bit mask (lo, hi clamped to [0, 32]).
__device__ __forceinline__ uint32_t bit_range(int lo, int hi) {
  lo = min(max(lo, 0), 32);
  hi = min(max(hi, 0), 32);
  if (hi <= lo) return 0u;
  const uint32_t upto_hi = hi == 32 ? 0xFFFFFFFFu : ((1u << hi) - 1u);
  const uint32_t below_lo = lo == 32 ? 0xFFFFFFFFu : ((1u << lo) - 1u);
  return upto_hi & ~below_lo;
}

__device__ __noinline__ void pair_add(const GrepWork& w, uint32_t f, uint32_t k, uint64_t cnt) {
  const uint64_t key = ((uint64_t)f << 32) | k;
  uint64_t slot = splitmix64(key) & w.pair_mask;
  // a run this long means the table is (nearly) full: report it rather than
  // walk the whole table for every add
  const uint64_t limit = w.pair_mask < 4095 ? w.pair_mask : 4095;
  for (uint64_t probe = 0; probe <= limit; ++probe, slot = (slot + 1) & w.pair_mask) {
    const unsigned long long cur = atomicCAS((unsigned long long*)&w.pair[2 * slot], (unsigned long long)kPairEmpty,
                                             (unsigned long long)key);
    if (cur == kPairEmpty || cur == key) {
      atomicAdd((unsigned long long*)&w.pair[2 * slot + 1], (unsigned long long)cnt);
      if (cur == kPairEmpty) {  // a new pair: its 256-slot region is one compact must visit
        const uint64_t r = slot >> 8;
        const uint32_t bit = 1u << (r & 31);
        if (!(*(volatile uint32_t*)&w.ptouch[r >> 5] & bit)) atomicOr(&w.ptouch[r >> 5], bit);
      }
      return;
    }
  }
  set_err(w, -ENOSPC);
}

// Space for n <= kRecPage records in the calling block's current output page
// (a new page when it does not fit); run by one thread, page state in shared
// memory. Returns the pool index of the first record, or ~0 when out of pages.
__device__ uint64_t rec_reserve(const GrepWork& w, uint32_t n, uint32_t* page_s, uint32_t* used_s) {
  if (*page_s == kNoPage || *used_s + n > kRecPage) {
    if (*page_s != kNoPage) w.page_used[*page_s] = *used_s;
    const unsigned long long p = atomicAdd(&w.vars[V_NPAGES], 1ull);
    if (p >= w.max_pages) {
      set_err(w, -ENOSPC);
      *page_s = kNoPage;
      return ~0ull;
    }
    *page_s = (uint32_t)p;
    *used_s = 0;
  }
  const uint64_t base = (uint64_t)*page_s * kRecPage + *used_s;
  *used_s += n;
  return base;
}
__device__ __forceinline__ void rec_close(const GrepWork& w, uint32_t page, uint32_t used) {
  if (page != kNoPage) w.page_used[page] = used;
}

struct ScanAcc {
  uint64_t dsum, dxor, nh;
};

// Count table slots per block: the distinct words of one item (a 16 KiB chunk
// of the C4 corpus has ~450, a 256 KiB file ~3000); an item that exhausts the
// 64-probe limit spills to the global (file, word) table (still exact)
constexpr uint32_t kMaxCountSlots = 4096;  // (runtime: GrepWork.cslots, a power of two)
static_assert(kRecPage >= kMaxCountSlots, "one item's records fit one record page");
// Shared-memory state of one scan block (dynamic shared memory, see scan_smem).
struct ScanSmem {
  uint8_t* buf;     // kPre + chunk + kHalo + kSlack bytes; file byte p at buf[kPre + p - s]
  uint32_t* mask;   // word-byte bits per 32-byte stripe of buf (+1 zero stripe)
  uint32_t* ckey;   // count table: word + 1 (0 = empty)
  uint32_t* ccnt;
  uint32_t* occ;    // occupied count slots, one bit each
  uint64_t hf;      // splitmix64(file index) of the current item (digest)
  uint32_t cmask;   // count table slots - 1
};

// One hit of word k at file position pos: per-item shared count (spilling to
// the global table when the probe run is exhausted), digest, optional hit list.
// shared-memory atomics by address space (a generic atomic on a shared
// address is slower than ATOMS)
__device__ __forceinline__ uint32_t atoms_cas(uint32_t* p, uint32_t cmp, uint32_t v) {
  uint32_t r;
  asm volatile("atom.shared.cas.b32 %0, [%1], %2, %3;" : "=r"(r) : "r"(detail::smem_u32(p)), "r"(cmp), "r"(v)
               : "memory");
  return r;
}
__device__ __forceinline__ void reds_add(uint32_t* p, uint32_t v) {
  asm volatile("red.shared.add.u32 [%0], %1;" ::"r"(detail::smem_u32(p)), "r"(v) : "memory");
}
__device__ __forceinline__ void reds_or(uint32_t* p, uint32_t v) {
  asm volatile("red.shared.or.b32 [%0], %1;" ::"r"(detail::smem_u32(p)), "r"(v) : "memory");
}
__device__ __forceinline__ uint32_t lds_u32(const uint32_t* p) {
  uint32_t v;
  asm volatile("ld.shared.u32 %0, [%1];" : "=r"(v) : "r"(detail::smem_u32(p)) : "memory");
  return v;
}

// The rare per-hit paths, out of line (the token loop keeps its registers).
__device__ __noinline__ void hit_spill(const GrepWork& w, uint32_t f, uint32_t k, uint32_t* spilled) {
  pair_add(w, f, k, 1);  // this item's records then all go through the global table
  *spilled = 1;
}
__device__ __noinline__ void hit_list(const GrepWork& w, uint32_t f, uint32_t k, uint64_t pos, uint64_t* hits,
                                      uint64_t hit_cap) {
  const unsigned long long idx = atomicAdd(&w.vars[V_NLISTED], 1ull);
  if (idx < hit_cap) {
    hits[2 * idx] = ((uint64_t)f << 32) | k;
    hits[2 * idx + 1] = pos;
  }
}

// One hit of word k at file position pos: per-item shared count (spilling to
// the global table when the probe run is exhausted), digest, optional hit list.
__device__ __forceinline__ void count_hit(const GrepWork& w, const ScanSmem& S, uint32_t* spilled,
                                          uint32_t f, uint32_t k, uint64_t pos, uint64_t* hits, uint64_t hit_cap,
                                          ScanAcc& acc) {
  uint32_t cs = (k * 2654435761u) & S.cmask;
  bool done = false;
  for (uint32_t p = 0; p < 64; ++p, cs = (cs + 1) & S.cmask) {
    uint32_t prev = lds_u32(&S.ckey[cs]);  // a word seen before in this item: no atomic on the key
    if (prev == 0) {
      prev = atoms_cas(&S.ckey[cs], 0u, k + 1);
      if (prev == 0) reds_or(&S.occ[cs >> 5], 1u << (cs & 31));
    }
    if (prev == 0 || prev == k + 1) {
      reds_add(&S.ccnt[cs], 1u);
      done = true;
      break;
    }
  }
  if (!done) hit_spill(w, f, k, spilled);
  const uint64_t m = hit_mix_hf(S.hf, pos, k);
  acc.dsum += m;
  acc.dxor ^= m;
  ++acc.nh;
  if (hits) hit_list(w, f, k, pos, hits, hit_cap);
}

// The next table entry at or after (bucket b, entry q) whose key (fingerprint
// + length) is `want`: returns it and advances (b, q) past it, or returns 0
// at the first empty entry (insertion filled the first empty slot in probe
// order and nothing is ever removed, so an empty slot ends the search). The
// caller verifies a candidate with ONE copy of its compare-and-count code
// (a match found in entry 0..3 of a bucket takes the same path: no warp
// divergence on the entry position).
__device__ __forceinline__ uint64_t next_candidate(const GrepWork& w, uint64_t want, uint32_t& b, uint32_t& q) {
  const uint32_t want_hi = (uint32_t)(want >> 6), want_len = (uint32_t)want & 63u;
  for (;;) {
    const uint4* bp = (const uint4*)&w.table[b];
    const uint4 e01 = __ldg(bp), e23 = __ldg(bp + 1);
    const uint32_t lo[4] = {e01.x, e01.z, e23.x, e23.z}, hi[4] = {e01.y, e01.w, e23.y, e23.w};
    // 4-bit masks of key matches and of empty entries; the first of either at
    // or after q decides (key_bits: fingerprint = hi & 0x7fffffff, length =
    // lo bits 26..31; an empty entry is all zero)
    uint32_t mm = 0, em = 0;
#pragma unroll
    for (int e = 0; e < 4; ++e) {
      mm |= (uint32_t)((hi[e] & 0x7FFFFFFFu) == want_hi && (lo[e] >> 26) == want_len && (lo[e] | hi[e])) << e;
      em |= (uint32_t)((lo[e] | hi[e]) == 0) << e;
    }
    const uint32_t sel = (mm | em) & (0xFu << q);
    if (sel) {
      const uint32_t e = __ffs(sel) - 1;
      if ((em >> e) & 1u) return 0;
      const uint64_t cand = ((uint64_t)(e & 2 ? (e & 1 ? hi[3] : hi[2]) : (e & 1 ? hi[1] : hi[0])) << 32) |
                            (e & 2 ? (e & 1 ? lo[3] : lo[2]) : (e & 1 ? lo[1] : lo[0]));
      q = e + 1;
      if (q == 4) {
        q = 0;
        b = (b + 4) & w.table_mask;
      }
      return cand;
    }
    q = 0;
    b = (b + 4) & w.table_mask;
  }
}

// One token: bytes buf[i, i + L), file position pos, 1 <= L <= 32.
__device__ __forceinline__ void scan_token(const GrepWork& w, const ScanSmem& S, uint32_t* spilled,
                                           uint32_t f, uint32_t i, uint32_t L, uint64_t pos, uint64_t* hits,
                                           uint64_t hit_cap, ScanAcc& acc) {
  // first 8 bytes: three aligned words and two funnel shifts
  const uint32_t* a = (const uint32_t*)(S.buf + (i & ~3u));
  const uint32_t a0 = a[0], a1 = a[1], a2 = a[2], r8 = (i & 3u) * 8;
  const uint32_t w0 = low_bytes(__funnelshift_r(a0, a1, r8), min((int)L, 4));
  const uint32_t w1 = low_bytes(__funnelshift_r(a1, a2, r8), min(max((int)L - 4, 0), 4));
  const uint64_t h = tok_hash(w0, w1, L);
  const uint32_t fi = filter_index(h, w.filt_log2);
  if (!((ld_filter(&w.filt[fi >> 5]) >> (fi & 31)) & 1u)) return;
  const uint64_t want = entry_key(h, L) >> 26;
  uint32_t b = (uint32_t)h & w.table_mask & ~3u, q = 0;
  for (;;) {
    const uint64_t ent = next_candidate(w, want, b, q);
    if (!ent) return;
    const uint32_t kp = (uint32_t)(ent & ((1u << 26) - 1)) - 1;
    const uint4* dw = (const uint4*)(w.dict + (size_t)kp * 32);  // padded slot (k_grep_dict)
    const uint4 d0 = __ldg(dw), d1 = __ldg(dw + 1);
    uint32_t v[8];  // the whole token, zero-padded: only gathered on a key match
    token_words(S.buf, i, L, v);
    const bool same = ((d0.x ^ v[0]) | (d0.y ^ v[1]) | (d0.z ^ v[2]) | (d0.w ^ v[3]) | (d1.x ^ v[4]) |
                       (d1.y ^ v[5]) | (d1.z ^ v[6]) | (d1.w ^ v[7])) == 0;
    if (same) {
      count_hit(w, S, spilled, f, kp, pos, hits, hit_cap, acc);
      if (ent & kDupBit) {  // the word's duplicates each count (R14)
        for (uint32_t d = w.dup_head[kp]; d; d = w.dup_next[d - 1])
          count_hit(w, S, spilled, f, d - 1, pos, hits, hit_cap, acc);
      }
      return;
    }
  }
}

// The byte ranges of chunk ci of item d: token starts in [s, e) count, [ws, we)
// is read (the chunk with up to kPre bytes before and kHalo after).
struct StepRange {
  uint64_t s, e, ws, we;
};
__device__ __forceinline__ StepRange step_range(const ItemDesc& d, uint32_t ci, uint32_t chunk) {
  StepRange r;
  if ((d.meta >> 30) & 1u) {  // multi-chunk whole file: rlen is its size
    r.s = (uint64_t)ci * chunk;
    r.e = min((uint64_t)d.rlen, r.s + chunk);
    r.ws = r.s >= kPre ? r.s - kPre : 0;
    r.we = min((uint64_t)d.rlen, r.e + kHalo);
  } else if (d.meta >> 31) {  // one-chunk file
    r.s = r.ws = 0;
    r.e = r.we = d.rlen;
  } else {  // a chunk of a larger file
    r.ws = d.roff;
    r.we = r.ws + d.rlen;
    r.s = r.ws + (d.meta & 31u);
    r.e = r.s + d.body;
  }
  return r;
}
__device__ __forceinline__ uint32_t item_chunks(const ItemDesc& d) { return ((d.meta >> 30) & 1u) ? d.body : 1u; }

// Persistent blocks pull items; an item is one chunk of a large file, a
// one-chunk file, or a multi-chunk file of at most whole_max bytes that the
// block scans chunk after chunk, counting in shared memory across chunks.
// Thread 0 claims the next item and loads its descriptor while the block
// works on the current one (the claim and the descriptor load are off the path).
__global__ void __launch_bounds__(256, 3) k_grep_scan(const __grid_constant__ gfs_ctx cv_, const __grid_constant__ GrepWork w, uint32_t chunk, uint64_t* hits,
                                                   uint64_t hit_cap, uint64_t* totals, uint32_t* rec,
                                                   uint64_t rec_cap) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  extern __shared__ __align__(16) uint8_t sm[];
  const int tid = threadIdx.x, nthr = blockDim.x, lane = tid & 31, wid = tid >> 5;
  const uint32_t buf_bytes = (kPre + chunk + kHalo + kSlack + 15) & ~15u;
  const uint32_t nstripe_max = (kPre + chunk + kHalo + 31) / 32;
  ScanSmem S;
  S.buf = sm;
  S.mask = (uint32_t*)(sm + buf_bytes);
  S.ckey = S.mask + ((nstripe_max + 1 + 3) & ~3u);
  const uint32_t cslots = w.cslots;
  S.ccnt = S.ckey + cslots;
  S.occ = S.ccnt + cslots;
  S.cmask = cslots - 1;
  uint16_t* tok = (uint16_t*)(S.occ + cslots / 32);  // token starts of one round (<= 32 per thread);
                                                          // in the flush: the occupied slots
  const uint32_t round_stripes = 2u * (uint32_t)nthr;
  __shared__ ItemDesc nd;  // the next item (claimed by thread 0 one item ahead)
  __shared__ unsigned long long nxt_item;
  __shared__ uint32_t page_s, used_s;
  __shared__ uint32_t spilled_s;
  __shared__ uint32_t warp_tot[32];
  __shared__ unsigned long long rbase_s;
  __shared__ unsigned long long nitems_s;
  ScanAcc acc{0, 0, 0};
  auto prefetch = [&]() {
    const uint64_t it = atomicAdd(&w.vars[V_NEXT], 1ull);
    nxt_item = it;
    if (it < nitems_s) nd = w.desc[it];
  };
  for (uint32_t i = tid; i < cslots; i += nthr) {  // dynamic smem is not cleared between launches
    S.ckey[i] = 0;
    S.ccnt[i] = 0;
  }
  for (uint32_t i = tid; i < cslots / 32; i += nthr) S.occ[i] = 0;
  if (tid == 0) {
    uint64_t ni = count_items(w);
    if (ni > w.max_items) {
      set_err(w, -ENOSPC);
      ni = w.max_items;
    }
    if (blockIdx.x == 0) w.vars[V_NITEMS] = ni;
    nitems_s = ni;
    page_s = kNoPage;
    used_s = 0;
    prefetch();
  }
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
    if (nxt_item >= nitems_s) break;
    const ItemDesc d = nd;
    const uint32_t f = d.gid;
    S.hf = splitmix64(f);
    const bool whole = d.meta >> 31;
    const uint32_t nch = item_chunks(d);
    if (tid == 0) spilled_s = 0;
    bool bad = false;
    for (uint32_t ci = 0; ci < nch; ++ci) {
      const StepRange r = step_range(d, ci, chunk);
      // file byte p lands at buf[kPre + p - s]; (dst - ws) % 16 == 0, so gread
      // moves the span with TMA (s is a multiple of the chunk, itself of 16)
      const uint32_t vlo = (uint32_t)(kPre - (r.s - r.ws)), vhi = vlo + (uint32_t)(r.we - r.ws);
      // (a lane-parallel gread_lanes by warp 0 measured slower here: 23 % vs 18 % of the item time)
      const int64_t got = gread(c, d.fd, r.ws, r.we - r.ws, S.buf + vlo);  // starts with a barrier
      lap(1);  // 1: gread
      if (got != (int64_t)(r.we - r.ws)) {  // the same value in every thread
        if (tid == 0) set_err(w, got < 0 ? got : -EIO);
        bad = true;
        break;
      }
      // pass 1: word-byte bits per 32-byte stripe; bytes outside [vlo, vhi) are non-word
      const uint32_t nstripe = (vhi + 31) / 32;
      for (uint32_t j = tid; j < nstripe; j += nthr)
        S.mask[j] = word_bits32(S.buf + 32 * j) & bit_range((int)vlo - 32 * (int)j, (int)vhi - 32 * (int)j);
      if (tid == 0) S.mask[nstripe] = 0;
      __syncthreads();
      lap(2);  // 2: pass 1
      if (tid == 0 && ci + 1 == nch) prefetch();  // next item's descriptor, overlapping pass 2
      // pass 2, by rounds of 2 stripes per thread: the starts of tokens in
      // [s, e) = buf[kPre, kPre + e - s) are compacted into `tok`, then every
      // thread takes every nthr-th token (balanced whatever the text layout)
      const uint32_t olo = kPre, ohi = kPre + (uint32_t)(r.e - r.s);
      const uint32_t jlo = olo / 32, jhi = (ohi - 1) / 32;
      const uint64_t pos0 = r.s - kPre;
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
            scan_token(w, S, &spilled_s, f, i, L, pos0 + i, hits, hit_cap, acc);
        }
        lap(4);  // 4: own tokens
        __syncthreads();  // tok and warp_tot are reused by the next round
        lap(5);  // 5: waiting for the block's other tokens
      }
    }
    if (bad && tid == 0) prefetch();  // (a failed read stops before the prefetch of the last chunk)
    // flush. The occupied slots, from the bitmap, into `tok` (free now)
    const uint32_t nwords = cslots / 32;
    const uint32_t wpt = (nwords + nthr - 1) / nthr, q0 = tid * wpt, q1 = min(q0 + wpt, nwords);
    uint32_t cnt = 0;
    for (uint32_t q = q0; q < q1; ++q) cnt += __popc(S.occ[q]);
    uint32_t incl = cnt;
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t t = __shfl_up_sync(0xFFFFFFFFu, incl, o);
      if (lane >= o) incl += t;
    }
    if (lane == 31) warp_tot[wid] = incl;
    __syncthreads();
    uint32_t off = incl - cnt, nocc = 0;
    for (int q = 0; q < (nthr >> 5); ++q) {
      const uint32_t t = warp_tot[q];
      off += q < wid ? t : 0u;
      nocc += t;
    }
    for (uint32_t q = q0; q < q1; ++q) {
      for (uint32_t x = S.occ[q]; x; x &= x - 1) tok[off++] = (uint16_t)(32 * q + __ffs(x) - 1);
      S.occ[q] = 0;
    }
    // a whole-file item with no spill owns its records; otherwise merge
    const bool direct = whole && !spilled_s && rec;
    if (direct && tid == 0 && nocc && !bad) rbase_s = rec_reserve(w, nocc, &page_s, &used_s);
    __syncthreads();
    if (w.prof && tid == 0) atomicAdd(&w.prof[7], 1ull);  // 7: items
    for (uint32_t q = tid; q < nocc; q += nthr) {
      const uint32_t cs = tok[q];
      const uint32_t k = S.ckey[cs] - 1, cnt = S.ccnt[cs];
      S.ckey[cs] = 0;
      S.ccnt[cs] = 0;
      if (bad) continue;
      if (direct) {
        atomicAdd((unsigned long long*)&totals[k], (unsigned long long)cnt);
        if (rbase_s != ~0ull) {
          uint32_t* o = w.rpool + 3 * (rbase_s + q);
          o[0] = f;
          o[1] = k;
          o[2] = cnt;
        }
      } else {
        pair_add(w, f, k, cnt);
      }
    }
    lap(6);  // 6: flush
  }
  if (tid == 0) rec_close(w, page_s, used_s);
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

// --------------------------------------------------------------- warp scan
// The warp-granularity scan (gfs_grep_params.scan = 1; the paper's API
// granularity is the warp): every warp pulls its own items and
// works through them with no block barrier. A warp maps the item's pages with
// gmmap_warp (zero copy: the text is read straight out of the cache frames,
// P:L426-441) and walks the item in 1 KiB steps, 32 bytes per lane:
//   - the next step's 32 bytes per lane are loaded while this step is scanned;
//   - each lane classifies its 32 bytes in registers (word_bits4), token
//     starts come from the masks and the previous lane's last bit (shuffle);
//   - the step (+ 64 lookahead bytes) is staged in the warp's shared buffer,
//     the token starts compacted into a list (warp prefix sum), and lanes take
//     every 32nd token: hash, L1 filter, one 32-byte bucket of the table, and
//     an exact 32-byte compare on a fingerprint match (as k_grep_scan);
//   - hits count in the warp's own shared table of packed (word + 1) << 16 |
//     count slots (an item has < 2^16 tokens, words < 65535), spilling to the
//     global (file, word) table when a probe run is exhausted;
//   - at the item's end a whole-file item writes its records straight into
//     the caller's array (one atomic per item reserves the space); chunks of
//     larger files merge through the (file, word) table.
constexpr uint32_t kWStep = 1024;            // bytes per warp step
constexpr uint32_t kWBuf = kWStep + 64;      // + lookahead (a token starting in the step reads <= 48 past it)
constexpr uint32_t kWTok = kWStep / 2;       // token starts per step at most
constexpr uint32_t kWProbe = 32;             // count-table probe run before a spill
struct WarpSmemLayout {
  static __host__ __device__ constexpr uint32_t buf() { return 0; }
  static __host__ __device__ constexpr uint32_t mask() { return kWBuf + 16; }
  static __host__ __device__ constexpr uint32_t tok() { return mask() + 36 * 4; }
  static __host__ __device__ constexpr uint32_t tab() { return tok() + kWTok * 2; }
  static __host__ __device__ constexpr uint32_t bytes(uint32_t slots) { return tab() + slots * 4; }
};

__device__ __forceinline__ uint32_t word_bits32_regs(uint4 a, uint4 b) {
  return word_bits4(a.x) | (word_bits4(a.y) << 4) | (word_bits4(a.z) << 8) | (word_bits4(a.w) << 12) |
         (word_bits4(b.x) << 16) | (word_bits4(b.y) << 20) | (word_bits4(b.z) << 24) | (word_bits4(b.w) << 28);
}
__device__ __forceinline__ uint32_t atoms_cas32(uint32_t* p, uint32_t cmp, uint32_t v) {
  uint32_t r;
  asm volatile("atom.shared.cas.b32 %0, [%1], %2, %3;" : "=r"(r) : "r"(detail::smem_u32(p)), "r"(cmp), "r"(v)
               : "memory");
  return r;
}
__device__ __forceinline__ void reds_add32(uint32_t* p, uint32_t v) {
  asm volatile("red.shared.add.u32 [%0], %1;" ::"r"(detail::smem_u32(p)), "r"(v) : "memory");
}

// One hit of word k in the warp's count table; false when the probe run is
// exhausted (the caller spills the hit to the (file, word) table).
__device__ __forceinline__ bool wcount(uint32_t* tab, uint32_t tmask, uint32_t k) {
  const uint32_t key = (k + 1) << 16;
  uint32_t s = (k * 2654435761u) & tmask;
  for (uint32_t p = 0; p < kWProbe; ++p, s = (s + 1) & tmask) {
    uint32_t v = lds_u32(&tab[s]);
    if (v == 0) {
      v = atoms_cas32(&tab[s], 0u, key | 1u);
      if (v == 0) return true;
    }
    if ((v & 0xFFFF0000u) == key) {
      reds_add32(&tab[s], 1u);
      return true;
    }
  }
  return false;
}

struct WHit {
  uint64_t dsum, dxor, nh;
  uint32_t spilled;
};
__device__ __forceinline__ void whit(const GrepWork& w, uint32_t* tab, uint32_t tmask, uint32_t f, uint64_t hf,
                                     uint32_t k, uint64_t pos, uint64_t* hits, uint64_t hit_cap, WHit& a) {
  if (!wcount(tab, tmask, k)) {
    pair_add(w, f, k, 1);  // this item's records then all go through the global table
    a.spilled = 1;
  }
  const uint64_t m = hit_mix_hf(hf, pos, k);
  a.dsum += m;
  a.dxor ^= m;
  ++a.nh;
  if (hits) hit_list(w, f, k, pos, hits, hit_cap);
}

// The token's bytes buf[i, i + L) as 8 zero-padded words.
__device__ __forceinline__ void wtoken_words(const uint8_t* buf, uint32_t i, uint32_t L, uint32_t (&v)[8]) {
  token_words(buf, i, L, v);
}
__device__ __forceinline__ bool wsame(const GrepWork& w, uint32_t kp, const uint32_t (&v)[8]) {
  const uint4* dw = (const uint4*)(w.dict + (size_t)kp * 32);  // padded slot (k_grep_dict)
  const uint4 d0 = __ldg(dw), d1 = __ldg(dw + 1);
  return ((d0.x ^ v[0]) | (d0.y ^ v[1]) | (d0.z ^ v[2]) | (d0.w ^ v[3]) | (d1.x ^ v[4]) | (d1.y ^ v[5]) |
          (d1.z ^ v[6]) | (d1.w ^ v[7])) == 0;
}
// A hit of table entry `ent` (word kp, and its duplicates, R14).
__device__ __forceinline__ void whit_entry(const GrepWork& w, uint32_t* tab, uint32_t tmask, uint32_t f, uint64_t hf,
                                           uint64_t ent, uint64_t pos, uint64_t* hits, uint64_t hit_cap, WHit& a) {
  const uint32_t kp = (uint32_t)(ent & ((1u << 26) - 1)) - 1;
  whit(w, tab, tmask, f, hf, kp, pos, hits, hit_cap, a);
  if (ent & kDupBit)
    for (uint32_t d = w.dup_head[kp]; d; d = w.dup_next[d - 1]) whit(w, tab, tmask, f, hf, d - 1, pos, hits, hit_cap, a);
}
// One token buf[i, i + L) (1 <= L <= 32) at file position pos: hash, L1
// filter, one 32-byte bucket of the table per step, an exact compare on a key
// match (as scan_token).
__device__ __forceinline__ void wscan_token(const GrepWork& w, const uint8_t* buf, uint32_t* tab, uint32_t tmask,
                                            uint32_t f, uint64_t hf, uint32_t i, uint32_t L, uint64_t pos,
                                            uint64_t* hits, uint64_t hit_cap, WHit& a) {
  const uint32_t* qw = (const uint32_t*)(buf + (i & ~3u));
  const uint32_t a0 = qw[0], a1 = qw[1], a2 = qw[2], r8 = (i & 3u) * 8;
  const uint32_t w0 = low_bytes(__funnelshift_r(a0, a1, r8), min((int)L, 4));
  const uint32_t w1 = low_bytes(__funnelshift_r(a1, a2, r8), min(max((int)L - 4, 0), 4));
  const uint64_t h = tok_hash(w0, w1, L);
  const uint32_t fi = filter_index(h, w.filt_log2);
  if (!((ld_filter(&w.filt[fi >> 5]) >> (fi & 31)) & 1u)) return;
  const uint64_t want = entry_key(h, L) >> 26;
  uint32_t b = (uint32_t)h & w.table_mask & ~3u, q = 0;
  for (;;) {
    const uint64_t ent = next_candidate(w, want, b, q);
    if (!ent) return;
    uint32_t v[8];
    wtoken_words(buf, i, L, v);
    if (wsame(w, (uint32_t)(ent & ((1u << 26) - 1)) - 1, v)) {
      whit_entry(w, tab, tmask, f, hf, ent, pos, hits, hit_cap, a);
      return;
    }
  }
}

// 32 bytes of lane `lane` of the step at p (a 1 KiB-aligned frame address);
// zeros for lanes >= nl.
__device__ __forceinline__ void wload(const uint8_t* p, int lane, int nl, uint4& a, uint4& b) {
  if (p && lane < nl) {
    const uint4* q = (const uint4*)(p + 32 * lane);
    a = __ldcs(q);  // streamed: the step is read once (its bytes are staged in shared memory)
    b = __ldcs(q + 1);
  } else {
    a = make_uint4(0, 0, 0, 0);
    b = a;
  }
}

// gmmap_warp of one whole page, out of line (once per page: the scan loop
// keeps its registers and the kernel its instruction cache footprint).
__device__ __noinline__ const uint8_t* wmap_page(const gfs_ctx* c, int fd, uint64_t q, int* err) {
  uint64_t m = 0;
  return (const uint8_t*)gmmap_t<detail::WarpGroup>(c, nullptr, c->page_size, 0, 0, fd, q << c->page_shift, &m, err);
}
__device__ __noinline__ void wunmap_page(const gfs_ctx* c, const uint8_t* p) { gmunmap_warp(c, (void*)p, 1); }

// A warp's two most recent page mappings (gmmap_warp); pages only advance, so
// mapping a new page releases the older one. Warp-uniform.
struct WPageWin {
  uint64_t pg0 = ~0ull, pg1 = ~0ull;
  const uint8_t* pp0 = nullptr;
  const uint8_t* pp1 = nullptr;
  int err = 0;
  __device__ __forceinline__ const uint8_t* map(const gfs_ctx* c, int fd, uint64_t q) {
    if (pg0 == q) return pp0;
    if (pg1 == q) return pp1;
    if (err) return nullptr;
    const bool use0 = pg0 == ~0ull || (pg1 != ~0ull && pg0 < pg1);
    const uint8_t* old = use0 ? pp0 : pp1;
    if (old) wunmap_page(c, old);
    int er = 0;
    const uint8_t* p = wmap_page(c, fd, q, &er);
    if (!p) err = er ? er : -EIO;
    if (use0) {
      pg0 = p ? q : ~0ull;
      pp0 = p;
    } else {
      pg1 = p ? q : ~0ull;
      pp1 = p;
    }
    return p;
  }
  __device__ __forceinline__ void release(const gfs_ctx* c) {
    if (pp0) wunmap_page(c, pp0);
    if (pp1) wunmap_page(c, pp1);
  }
};

__global__ void __launch_bounds__(256) k_grep_wscan(const __grid_constant__ gfs_ctx cv_, const __grid_constant__ GrepWork w,
                                                    uint64_t* hits, uint64_t hit_cap, uint64_t* totals,
                                                    uint32_t* rec, uint64_t rec_cap) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  extern __shared__ __align__(16) uint8_t sm[];
  const int lane = threadIdx.x & 31, wid = threadIdx.x >> 5;
  const uint32_t slots = w.cslots, tmask = slots - 1;
  uint8_t* ws = sm + (size_t)wid * WarpSmemLayout::bytes(slots);
  uint8_t* buf = ws + WarpSmemLayout::buf();
  uint32_t* msk = (uint32_t*)(ws + WarpSmemLayout::mask());
  uint16_t* tok = (uint16_t*)(ws + WarpSmemLayout::tok());
  uint32_t* tab = (uint32_t*)(ws + WarpSmemLayout::tab());
  const uint32_t shift = c->page_shift;
  const uint64_t P = c->page_size;
  for (uint32_t i = lane; i < slots; i += 32) tab[i] = 0;  // dynamic smem is not cleared between launches
  uint64_t nitems = count_items(w);
  if (nitems > w.max_items) {
    if (blockIdx.x == 0 && threadIdx.x == 0) set_err(w, -ENOSPC);
    nitems = w.max_items;
  }
  if (blockIdx.x == 0 && threadIdx.x == 0) w.vars[V_NITEMS] = nitems;
  WHit acc{0, 0, 0, 0};
  unsigned long long it = 0;
  if (lane == 0) it = atomicAdd(&w.vars[V_NEXT], 1ull);
  it = __shfl_sync(0xFFFFFFFFu, it, 0);
  while (it < nitems) {
    const ItemDesc d = w.desc[it];
    unsigned long long nxt = 0;
    if (lane == 0) nxt = atomicAdd(&w.vars[V_NEXT], 1ull);  // the next item's claim flies meanwhile
    const uint32_t f = d.gid;
    const uint64_t hf = splitmix64(f);
    const bool whole = d.meta >> 31;
    const int fd = d.fd;
    // token starts counted in [s, e); bytes read [s - 1, min(S, e + 33))
    uint64_t s, e, S;
    if (whole) {
      s = 0;
      e = S = d.rlen;
    } else {
      s = d.roff + (d.meta & 31u);
      e = s + d.body;
      S = w.size[d.f];
    }
    const uint64_t need_end = min(S, e + 33);
    // two-page window of gmmap_warp mappings (pages only ever advance)
    WPageWin pw;
    uint32_t prev = 0;  // W(t[x - 1]) for the current step x
    if (s > 0) {
      const uint8_t* p = pw.map(c, fd, (s - 1) >> shift);
      if (p) prev = is_word(p[(s - 1) & (P - 1)]) ? 1u : 0u;  // the same byte in every lane
    }
    uint64_t x = s;
    uint4 ca, cb, na, nb;
    {
      const uint8_t* p = pw.map(c, fd, x >> shift);
      wload(p ? p + (x & (P - 1)) : nullptr, lane, 32, ca, cb);
    }
    while (!pw.err && x < e) {
      const uint64_t nx = x + kWStep;
      // the next step: all of it if tokens start there, else the lookahead lanes
      const uint8_t* np = nullptr;
      int nl = 0;
      if (nx < need_end) {
        np = pw.map(c, fd, nx >> shift);
        nl = nx < e ? 32 : 2;
      }
      wload(np ? np + (nx & (P - 1)) : nullptr, lane, nl, na, nb);
      if (pw.err) break;
      // stage this step (+ the next step's first 64 bytes) for the token gathers
      *(uint4*)(buf + 32 * lane) = ca;
      *(uint4*)(buf + 32 * lane + 16) = cb;
      // word-byte masks; bytes at or past EOF are non-word
      const uint64_t lb = x + 32 * (uint64_t)lane;
      uint32_t m = word_bits32_regs(ca, cb);
      if (lb + 32 > S) m &= lb >= S ? 0u : ((1u << (uint32_t)(S - lb)) - 1u);
      msk[lane] = m;
      if (lane < 2) {
        *(uint4*)(buf + kWStep + 32 * lane) = na;
        *(uint4*)(buf + kWStep + 32 * lane + 16) = nb;
        const uint64_t lnb = nx + 32 * (uint64_t)lane;
        uint32_t mn = word_bits32_regs(na, nb);
        if (lnb + 32 > S) mn &= lnb >= S ? 0u : ((1u << (uint32_t)(S - lnb)) - 1u);
        msk[32 + lane] = mn;
      }
      // token starts in [x, e): W(t[i]) and not W(t[i - 1])
      const uint32_t up = __shfl_up_sync(0xFFFFFFFFu, m, 1);
      const uint32_t pl = lane ? (up >> 31) : prev;
      uint32_t st = m & ~((m << 1) | pl);
      if (lb + 32 > e) st &= lb >= e ? 0u : ((1u << (uint32_t)(e - lb)) - 1u);
      prev = __shfl_sync(0xFFFFFFFFu, m, 31) >> 31;
      const uint32_t cnt = __popc(st);
      uint32_t incl = cnt;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const uint32_t t = __shfl_up_sync(0xFFFFFFFFu, incl, o);
        if (lane >= o) incl += t;
      }
      const uint32_t total = __shfl_sync(0xFFFFFFFFu, incl, 31);
      uint32_t o = incl - cnt;
      for (uint32_t y = st; y; y &= y - 1) tok[o++] = (uint16_t)(32 * lane + __ffs(y) - 1);
      __syncwarp();
      for (uint32_t q = lane; q < total; q += 32) {
        const uint32_t i = tok[q], j = i >> 5, b = i & 31;
        const uint64_t win = ((uint64_t)msk[j + 1] << 32) | msk[j];
        const uint32_t L = __ffsll(~(win >> b)) - 1;  // >= 33: too long for any word (R12)
        if (L <= 32) wscan_token(w, buf, tab, tmask, f, hf, i, L, x + i, hits, hit_cap, acc);
      }
      __syncwarp();  // buf / msk / tok are rewritten by the next step
      ca = na;
      cb = nb;
      x = nx;
    }
    pw.release(c);
    const int err = pw.err;
    if (err && lane == 0) set_err(w, err);
    // flush: the warp's occupied slots -> records (direct) or the (file, word) table
    const bool direct = whole && !__any_sync(0xFFFFFFFFu, acc.spilled) && rec && !err;
    acc.spilled = 0;
    uint32_t nocc = 0;
    for (uint32_t i = lane; i < slots; i += 32) nocc += tab[i] != 0;
    unsigned long long base = 0;
    if (direct) {
      uint32_t inc = nocc;
#pragma unroll
      for (int o2 = 1; o2 < 32; o2 <<= 1) {
        const uint32_t t = __shfl_up_sync(0xFFFFFFFFu, inc, o2);
        if (lane >= o2) inc += t;
      }
      const uint32_t all = __shfl_sync(0xFFFFFFFFu, inc, 31);
      if (lane == 31 && all) base = atomicAdd(&w.vars[V_NDIRECT], (unsigned long long)all);
      base = __shfl_sync(0xFFFFFFFFu, base, 31) + (inc - nocc);
    }
    for (uint32_t i = lane; i < slots; i += 32) {
      const uint32_t v = tab[i];
      if (!v) continue;
      tab[i] = 0;
      if (err) continue;
      const uint32_t k = (v >> 16) - 1, n = v & 0xFFFFu;
      if (direct) {
        atomicAdd((unsigned long long*)&totals[k], (unsigned long long)n);
        if (base < rec_cap) {
          uint32_t* r = rec + 3 * base;
          r[0] = f;
          r[1] = k;
          r[2] = n;
        }
        ++base;
      } else {
        pair_add(w, f, k, n);
      }
    }
    __syncwarp();
    it = __shfl_sync(0xFFFFFFFFu, nxt, 0);
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

__global__ void k_grep_close(const __grid_constant__ gfs_ctx cv_, const __grid_constant__ GrepWork w) {
  const gfs_ctx* c = &cv_;  // by value: the context's fields come from the constant bank
  const uint32_t nfiles = (uint32_t)w.vars[V_NFILES];
  for (uint32_t f = blockIdx.x; f < nfiles; f += gridDim.x) {
    const int fd = w.fd[f];
    if (fd >= 0) gclose(c, fd);
  }
}

// Records of the (file, word) table (chunked files, spilled items) + their
// word totals. A block takes 2048 consecutive slots (8 per thread, 128
// contiguous bytes), reserves output space for the valid ones in its record
// page, and empties the slots again for the next run.
__global__ void __launch_bounds__(256) k_grep_compact(const __grid_constant__ GrepWork w, int want_rec,
                                                      uint64_t* totals) {
  __shared__ uint32_t warp_tot[8];
  __shared__ uint32_t page_s, used_s;
  __shared__ unsigned long long base_s;
  const int tid = threadIdx.x, lane = tid & 31, wid = tid >> 5;
  if (tid == 0) {
    page_s = kNoPage;
    used_s = 0;
  }
  const uint64_t n = w.pair_mask + 1;  // a power of two >= 1024
  constexpr int kPer = 8;                // slots per thread (128 bytes in flight per thread)
  for (uint64_t blk = blockIdx.x; blk * 256 * kPer < n; blk += gridDim.x) {
    // the 8 regions of 256 slots this block covers (one per warp): only the
    // ones a pair was inserted into this run are read
    const uint32_t tb = (w.ptouch[blk >> 2] >> ((blk & 3) * 8)) & 0xFFu;
    if (!tb) continue;  // (the same for every thread of the block)
    const bool mine = (tb >> wid) & 1u;
    const uint64_t i0 = blk * 256 * kPer + (uint64_t)tid * kPer;
    uint4* src = (uint4*)(w.pair + 2 * i0);
    uint64_t key[kPer], cnt[kPer];
    uint32_t nv = 0;
#pragma unroll
    for (int q = 0; q < kPer; ++q) {
      const uint4 v = (mine && i0 < n) ? src[q] : make_uint4(0xFFFFFFFFu, 0xFFFFFFFFu, 0u, 0u);  // (n >= 1024: whole groups)
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
    if (tid == 0) base_s = (all && want_rec) ? rec_reserve(w, all, &page_s, &used_s) : ~0ull;
    __syncthreads();
    uint64_t idx = base_s + before + incl - nv;
#pragma unroll
    for (int q = 0; q < kPer; ++q) {
      if (key[q] == kPairEmpty) continue;
      const uint32_t k = (uint32_t)key[q];
      atomicAdd((unsigned long long*)&totals[k], (unsigned long long)cnt[q]);
      if (base_s != ~0ull) {
        uint32_t* o = w.rpool + 3 * idx;
        o[0] = (uint32_t)(key[q] >> 32);
        o[1] = k;
        o[2] = (uint32_t)cnt[q];
      }
      ++idx;
      src[q] = make_uint4(0xFFFFFFFFu, 0xFFFFFFFFu, 0u, 0u);  // empty again for the next run
    }
    if (tid == 0) atomicAnd(&w.ptouch[blk >> 2], ~(0xFFu << ((blk & 3) * 8)));  // regions empty again
    __syncthreads();  // warp_tot / base_s reuse
  }
  if (tid == 0) rec_close(w, page_s, used_s);
}

// Pack the used part of every record page into d_rec: one block scans the
// page counts (k_grep_pack_scan), then a grid copies the pages.
__global__ void k_grep_pack_scan(const __grid_constant__ GrepWork w, uint64_t rec_cap) {
  __shared__ uint64_t part[1024];
  const uint32_t tid = threadIdx.x, nthr = blockDim.x;
  const uint64_t np = min((uint64_t)w.vars[V_NPAGES], w.max_pages);
  const uint64_t per = (np + nthr - 1) / nthr;
  const uint64_t a = min(np, tid * per), b = min(np, a + per);
  uint64_t s = 0;
  for (uint64_t i = a; i < b; ++i) s += w.page_used[i];
  part[tid] = s;
  __syncthreads();
  if (tid == 0) {
    uint64_t run = w.vars[V_NDIRECT];  // the warp scan's direct records come first
    for (uint32_t q = 0; q < nthr; ++q) {
      const uint64_t v = part[q];
      part[q] = run;
      run += v;
    }
    w.vars[V_NREC] = run;
    if (run > rec_cap) set_err(w, -ENOSPC);
  }
  __syncthreads();
  uint64_t run = part[tid];
  for (uint64_t i = a; i < b; ++i) {
    w.page_base[i] = run;
    run += w.page_used[i];
  }
}

__global__ void k_grep_pack_copy(const __grid_constant__ GrepWork w, uint32_t* rec, uint64_t rec_cap) {
  const uint64_t np = min((uint64_t)w.vars[V_NPAGES], w.max_pages);
  for (uint64_t p = blockIdx.x; p < np; p += gridDim.x) {
    const uint64_t base = w.page_base[p];
    const uint64_t lim = base < rec_cap ? rec_cap - base : 0ull;
    const uint64_t n = (uint64_t)w.page_used[p] < lim ? (uint64_t)w.page_used[p] : lim;
    const uint32_t* src = w.rpool + 3 * (p * kRecPage);
    uint32_t* dst = rec + 3 * base;
    for (uint64_t i = threadIdx.x; i < 3 * n; i += blockDim.x) dst[i] = src[i];
  }
}

__global__ void k_grep_summary(const __grid_constant__ GrepWork w, uint64_t* out) {
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
    // compact emptied every used slot: the next run skips the full clear
    if (w.vars[V_ERR] == 0) w.keep[K_PAIRS] = kPairsClean;
  }
}

// Minimum batch-space weight of a whole-file item: chunk/16 rounded up to a
// stripe, so segments stay 32-byte aligned and a batch holds <= 17 items.
uint64_t pow2_at_least(uint64_t x) {
  uint64_t p = 1;
  while (p < x) p <<= 1;
  return p;
}

struct Layout {
  uint64_t off[19];
  uint64_t total;
  uint64_t max_items, tcap, pcap, max_pages;
  uint32_t flog2;
};

Layout layout(const gfs_grep_params* p) {
  Layout L{};
  L.tcap = pow2_at_least(p->max_words * 8ull < 1024 ? 1024 : p->max_words * 8ull);
  L.pcap = pow2_at_least(p->pair_cap < 1024 ? 1024 : p->pair_cap);
  // filter: >= 4.5 bits per word, 1 Ki .. 256 Ki bits (<= 32 KiB: it must stay in L1)
  L.flog2 = 10;
  while (L.flog2 < 18 && (1ull << L.flog2) < p->max_words * 9ull / 2) ++L.flog2;
  const uint64_t chunk = p->chunk ? p->chunk : 1;
  // items: one per chunk of corpus plus one partial chunk per file
  L.max_items = p->corpus_cap / chunk + p->max_files + 1;
  // record pages: the records themselves plus one partly used page per block
  // of the scan (<= 8 per SM) and of compact (4 per SM), 160 SMs at most
  L.max_pages = p->rec_cap / kRecPage + 160 * 12 + 2;
  const uint64_t sizes[] = {
      (uint64_t)p->max_words * 32,                         // 0 dict
      L.tcap * 8,                                          // 1 table
      (uint64_t)p->max_words * 4,                          // 2 dup_head
      (uint64_t)p->max_words * 4,                          // 3 dup_next
      p->list_cap + 64,                                    // 4 list
      (p->list_cap / kListChunk + 2) * 4,                  // 5 list_chunk
      (uint64_t)p->max_files * 8,                          // 6 line_off
      (uint64_t)p->max_files * 4,                          // 7 fd
      (uint64_t)p->max_files * 8,                          // 8 size
      L.max_items * sizeof(ItemDesc),                      // 9 desc
      L.pcap * 16,                                         // 10 pair
      L.max_pages * kRecPage * 12,                         // 11 record pages
      L.max_pages * 4,                                     // 12 page_used
      L.max_pages * 8,                                     // 13 page_base
      V_NVARS * 8,                                         // 14 vars
      K_NKEEP * 8,                                         // 15 keep (persistent)
      (1ull << L.flog2) / 8,                               // 16 word filter
      ptouch_words(L.pcap) * 4,                            // 17 touched regions of the pair table
  };
  uint64_t o = 0;
  for (int i = 0; i < 18; ++i) {
    L.off[i] = o;
    o += (sizes[i] + 255) & ~255ull;
  }
  L.total = o;
  return L;
}

uint32_t scan_smem(uint32_t chunk, uint32_t block, uint32_t cslots) {
  const uint32_t buf_bytes = (kPre + chunk + kHalo + kSlack + 15) & ~15u;
  const uint32_t nstripe_max = (kPre + chunk + kHalo + 31) / 32;
  const uint32_t tok_bytes = 64 * block > 2 * cslots ? 64 * block : 2 * cslots;
  return buf_bytes + ((nstripe_max + 1 + 3) & ~3u) * 4 + 2 * cslots * 4 + cslots / 8 + tok_bytes;
}

// Count slots per scan block: the most (<= 4096) that keep >= 768 threads of
// the scan resident per SM (latency hiding) in 227 KiB of shared memory.
uint32_t pick_cslots(uint32_t chunk, uint32_t block) {
  const uint32_t blocks = (768 + block - 1) / block;
  const uint32_t budget = 232448 / blocks - 1024 - 2048;  // per-block reserve + static shared memory
  uint32_t cs = kMaxCountSlots;
  while (cs > 512 && scan_smem(chunk, block, cs) > budget) cs >>= 1;
  return cs;
}

// Count-table slots per warp of the warp scan (a power of two; GFS_GREP_WSLOTS
// overrides it for tuning): 1024 hold the ~560 distinct words of a 32 KiB C4
// item at about half load and leave room for 24 warps per SM (2048 with 64 KiB
// items: 16 warps per SM, measured slower).
uint32_t wscan_slots() {
  uint32_t v = 1024;
  if (const char* e = getenv("GFS_GREP_WSLOTS")) {
    const long x = atol(e);
    if (x >= 256 && x <= 8192 && (x & (x - 1)) == 0) v = (uint32_t)x;
  }
  return v;
}

bool grep_params_ok(const gfs_grep_params* p) {
  if (!p || p->max_files == 0 || p->max_words == 0 || p->max_words >= (1u << 26) || p->chunk == 0 ||
      (p->chunk & 15) || p->grid == 0 || p->block == 0 || p->block > 256 || (p->block & 31) || p->scan > 1)
    return false;
  const bool wscan = p->scan == 1;
  if (!wscan && p->chunk + kPre + kHalo > 65536) return false;  // 16-bit token offsets into the item buffer
  // warp scan: 1 KiB steps never straddle a chunk; an item has < 2^16 tokens
  // and a word index fits the 16-bit key of a count slot
  if (wscan && ((p->chunk & (kWStep - 1)) || p->chunk > 65536 || p->whole_max > 65536 || p->max_words >= 65535))
    return false;
  return true;
}

std::string list_dir(const char* list_path) {
  const char* slash = strrchr(list_path, '/');
  std::string dir = slash ? std::string(list_path, (size_t)(slash - list_path)) : std::string(".");
  if (dir.empty()) dir = "/";  // a list at the root: "/" + "/" + line still resolves
  return dir;
}

// Everything one grep run enqueues on stream s, given the staged path strings
// (device memory) and the validated parameters: shared by gfs_grep and the
// CUDA-graph path (gfs_grep_graph), which captures exactly this sequence.
int grep_enqueue(gfs_handle* h, cudaStream_t s, const char* d_dict, const char* d_list, const char* d_dir,
                 uint32_t dir_len, const gfs_grep_params* p, void* d_work, uint32_t* d_rec, uint64_t rec_cap,
                 uint64_t* d_totals, uint64_t* d_hits, uint64_t* d_summary, unsigned long long* prof) {
  const bool wscan = p->scan == 1;
  const Layout L = layout(p);
  uint8_t* base = (uint8_t*)d_work;
  GrepWork w;
  w.dict = base + L.off[0];
  w.table = (uint64_t*)(base + L.off[1]);
  w.table_mask = (uint32_t)(L.tcap - 1);
  w.dup_head = (uint32_t*)(base + L.off[2]);
  w.dup_next = (uint32_t*)(base + L.off[3]);
  w.list = base + L.off[4];
  w.list_chunk = (uint32_t*)(base + L.off[5]);
  w.line_off = (uint64_t*)(base + L.off[6]);
  w.file_ids = p->file_ids;
  w.fd = (int32_t*)(base + L.off[7]);
  w.size = (uint64_t*)(base + L.off[8]);
  w.desc = (ItemDesc*)(base + L.off[9]);
  w.max_items = L.max_items;
  w.chunk = p->chunk;
  w.cslots = wscan ? wscan_slots() : pick_cslots(p->chunk, p->block);
  if (wscan) {
    // whole-file items up to whole_max (default: 2 chunks), counted by one warp
    const uint32_t wm = p->whole_max ? p->whole_max : 2 * p->chunk;
    const uint32_t wc = wm / p->chunk;
    w.whole_chunks = wc < kMaxWholeChunks ? wc : kMaxWholeChunks;
    if ((uint64_t)w.whole_chunks * p->chunk > 65536) w.whole_chunks = 65536 / p->chunk;
  } else {
    // default: what the count table holds (~64 text bytes per distinct word)
    const uint32_t wm = p->whole_max ? p->whole_max : w.cslots * 64u;
    const uint32_t wc = wm / p->chunk;
    w.whole_chunks = wc < kMaxWholeChunks ? wc : kMaxWholeChunks;
  }
  w.pair = (uint64_t*)(base + L.off[10]);
  w.pair_mask = L.pcap - 1;
  w.ptouch = (uint32_t*)(base + L.off[17]);
  w.rpool = (uint32_t*)(base + L.off[11]);
  w.page_used = (uint32_t*)(base + L.off[12]);
  w.page_base = (uint64_t*)(base + L.off[13]);
  w.max_pages = L.max_pages;
  w.vars = (unsigned long long*)(base + L.off[14]);
  w.keep = (unsigned long long*)(base + L.off[15]);
  w.filt = (uint32_t*)(base + L.off[16]);
  w.filt_log2 = L.flog2;

  const gfs_ctx c = gfs_launch::ctx_val(h);
  w.prof = prof;
  const uint32_t smem = wscan ? (p->block / 32) * WarpSmemLayout::bytes(w.cslots) : scan_smem(p->chunk, p->block, w.cslots);
  if (smem > 200 * 1024) return -EINVAL;
  if (wscan) cudaFuncSetAttribute(k_grep_wscan, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  else cudaFuncSetAttribute(k_grep_scan, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  int dev = 0, nsm = 148;
  cudaGetDevice(&dev);
  cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, dev);
  const uint64_t lb = p->list_cap / kListChunk + 1, lr = p->list_cap / kListRead + 1;
  const uint32_t list_blocks = (uint32_t)(lb < 1024 ? lb : 1024);
  // one opener per 64 KiB piece: a block that opens the list after all others
  // closed it would re-validate it with the host (close-to-open)
  const uint32_t read_blocks = (uint32_t)(lr < 1024 ? lr : 1024);
  k_grep_init<<<nsm * 4, 256, 0, s>>>(w, p->max_words);
  k_grep_hold<<<1, 32, 0, s>>>(c, d_dict, d_list, w, 0, (int)p->keep_open);
  k_grep_pairclear<<<nsm * 4, 256, 0, s>>>(w);
  k_grep_dict<<<nsm, 256, 0, s>>>(c, d_dict, w, p->max_words);
  k_grep_list_read<<<read_blocks, 256, 0, s>>>(c, d_list, w, p->list_cap);
  k_grep_list_count<<<list_blocks, 256, 0, s>>>(w);
  k_grep_list_scan<<<1, 1024, 0, s>>>(w, p->max_files);
  k_grep_list_emit<<<list_blocks, 256, 0, s>>>(w, p->max_files);
  // gopen is collective with one leader thread: many one-warp blocks keep
  // more opens in flight (host RPCs when cold, L2 round trips when warm)
  k_grep_open<<<nsm * 16, 32, 0, s>>>(c, w, d_dir, dir_len, p->max_files);
  k_grep_items<<<nsm * 2, 256, 0, s>>>(w);
  cudaMemsetAsync(d_totals, 0, (size_t)p->max_words * 8, s);
  // persistent scan grid: every resident block slot once (p->grid caps it)
  int occ = 1;
  if (wscan) cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, k_grep_wscan, (int)p->block, smem);
  else cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, k_grep_scan, (int)p->block, smem);
  const uint32_t scan_grid = (uint32_t)(occ > 0 ? occ : 1) * (uint32_t)nsm;
  if (wscan)
    k_grep_wscan<<<scan_grid < p->grid ? scan_grid : p->grid, p->block, smem, s>>>(
        c, w, d_hits, d_hits ? p->hit_cap : 0, d_totals, d_rec, d_rec ? rec_cap : 0);
  else
    k_grep_scan<<<scan_grid < p->grid ? scan_grid : p->grid, p->block, smem, s>>>(
        c, w, p->chunk, d_hits, d_hits ? p->hit_cap : 0, d_totals, d_rec, d_rec ? rec_cap : 0);
  if (!p->keep_open) k_grep_close<<<nsm * 16, 32, 0, s>>>(c, w);
  k_grep_compact<<<nsm * 4, 256, 0, s>>>(w, d_rec ? 1 : 0, d_totals);
  if (d_rec) {
    k_grep_pack_scan<<<1, 1024, 0, s>>>(w, rec_cap);
    k_grep_pack_copy<<<nsm * 8, 256, 0, s>>>(w, d_rec, rec_cap);
  }
  k_grep_hold<<<1, 32, 0, s>>>(c, d_dict, d_list, w, 1, (int)p->keep_open);
  k_grep_summary<<<1, 32, 0, s>>>(w, d_summary);
  return 0;
}

}  // namespace

GFS_API uint64_t gfs_grep_work_bytes(const gfs_grep_params* p) { return p ? layout(p).total : 0; }

GFS_API int gfs_grep(gfs_handle* h, void* stream, const char* dict_path, const char* list_path,
                     const gfs_grep_params* p, void* d_work, uint32_t* d_rec, uint64_t rec_cap, uint64_t* d_totals,
                     uint64_t* d_hits, uint64_t* d_summary) {
  if (!h || !dict_path || !list_path || !d_work || !d_totals || !d_summary || !grep_params_ok(p)) return -EINVAL;
  cudaStream_t s = (cudaStream_t)stream;
  // path arguments: dictionary, list, the list's directory (relative lines)
  gfs_launch::ArgStage as(h, s);
  const std::string dir = list_dir(list_path);
  const char* strs[3] = {dict_path, list_path, dir.c_str()};
  if (const int e = as.stage(strs, 3)) return e;
  const char* d_dict = as.str(0);
  const char* d_list = as.str(1);
  const char* d_dir = as.str(2);

  static unsigned long long* d_prof = nullptr;  // GFS_GREP_PROF=1 (diagnostics only)
  unsigned long long* prof = nullptr;
  if (getenv("GFS_GREP_PROF") && *getenv("GFS_GREP_PROF") == '1') {
    if (!d_prof && cudaMalloc((void**)&d_prof, 8 * sizeof(unsigned long long)) != cudaSuccess) d_prof = nullptr;
    if (d_prof) cudaMemsetAsync(d_prof, 0, 8 * sizeof(unsigned long long), s);
    prof = d_prof;
  }
  if (const int e = grep_enqueue(h, s, d_dict, d_list, d_dir, (uint32_t)dir.size(), p, d_work, d_rec, rec_cap,
                                 d_totals, d_hits, d_summary, prof))
    return e;
  if (prof) {
    unsigned long long pv[8];
    cudaMemcpyAsync(pv, prof, sizeof(pv), cudaMemcpyDeviceToHost, s);
    cudaStreamSynchronize(s);
    double tot = 0;
    for (int i = 0; i < 7; ++i) tot += (double)pv[i];
    tot += 1e-9;
    fprintf(stderr, "gfs_grep[scan prof, thread 0 cycles]: items=%llu loop-top=%.1f%% gread=%.1f%% pass1=%.1f%% "
            "toklist=%.1f%% tokens=%.1f%% wait-others=%.1f%% flush=%.1f%% (%.0f cycles/item)\n", pv[7],
            100 * pv[0] / tot, 100 * pv[1] / tot, 100 * pv[2] / tot, 100 * pv[3] / tot, 100 * pv[4] / tot,
            100 * pv[5] / tot, 100 * pv[6] / tot, tot / (double)(pv[7] ? pv[7] : 1));
  }
  const cudaError_t e = cudaGetLastError();
  if (e != cudaSuccess) fprintf(stderr, "gfs_grep: launch failed: %s\n", cudaGetErrorString(e));
  return e == cudaSuccess ? 0 : -EIO;
}

// ------------------------------------------------------------------ CUDA graph
// A grep run captured once as a CUDA graph and replayed: the pipeline is ~16
// small kernels, launch-bound for small corpora (C1). The path strings live in
// device memory the graph owns (not in the per-call argument slots), the
// parameters and the cache context are fixed at capture: re-create the graph
// after gfs_export / gfs_attach_peer or to change any argument.
struct gfs_grep_graph {
  cudaGraphExec_t exec = nullptr;
  char* d_str = nullptr;
  int device = 0;
};

GFS_API int gfs_grep_graph_create(gfs_handle* h, void* stream, const char* dict_path, const char* list_path,
                                  const gfs_grep_params* p, void* d_work, uint32_t* d_rec, uint64_t rec_cap,
                                  uint64_t* d_totals, uint64_t* d_hits, uint64_t* d_summary, gfs_grep_graph** out) {
  if (!h || !dict_path || !list_path || !d_work || !d_totals || !d_summary || !out || !grep_params_ok(p))
    return -EINVAL;
  const std::string dir = list_dir(list_path);
  const char* strs[3] = {dict_path, list_path, dir.c_str()};
  for (const char* x : strs)
    if (strlen(x) >= GFS_MAX_PATH) return -ENAMETOOLONG;
  int prev = 0;
  cudaGetDevice(&prev);
  auto* g = new gfs_grep_graph();
  g->device = gfs_internal_device(h);
  cudaSetDevice(g->device);
  char hs[3 * GFS_MAX_PATH] = {};
  for (int i = 0; i < 3; ++i) memcpy(hs + i * GFS_MAX_PATH, strs[i], strlen(strs[i]) + 1);
  cudaStream_t cs = nullptr;
  cudaGraph_t graph = nullptr;
  int rc = -EIO;
  if (cudaMalloc((void**)&g->d_str, sizeof(hs)) == cudaSuccess &&
      cudaMemcpy(g->d_str, hs, sizeof(hs), cudaMemcpyHostToDevice) == cudaSuccess &&
      cudaStreamCreateWithFlags(&cs, cudaStreamNonBlocking) == cudaSuccess &&
      cudaStreamBeginCapture(cs, cudaStreamCaptureModeRelaxed) == cudaSuccess) {
    const int e = grep_enqueue(h, cs, g->d_str, g->d_str + GFS_MAX_PATH, g->d_str + 2 * GFS_MAX_PATH,
                               (uint32_t)dir.size(), p, d_work, d_rec, rec_cap, d_totals, d_hits, d_summary, nullptr);
    const cudaError_t ec = cudaStreamEndCapture(cs, &graph);
    if (e) rc = e;
    else if (ec == cudaSuccess && graph && cudaGraphInstantiate(&g->exec, graph, 0) == cudaSuccess) rc = 0;
  }
  if (graph) cudaGraphDestroy(graph);
  if (cs) cudaStreamDestroy(cs);
  (void)cudaGetLastError();
  (void)stream;
  cudaSetDevice(prev);
  if (rc) {
    if (g->d_str) cudaFree(g->d_str);
    delete g;
    return rc;
  }
  *out = g;
  return 0;
}

GFS_API int gfs_grep_graph_launch(gfs_grep_graph* g, void* stream) {
  if (!g || !g->exec) return -EINVAL;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(g->device);
  const cudaError_t e = cudaGraphLaunch(g->exec, (cudaStream_t)stream);
  cudaSetDevice(prev);
  return e == cudaSuccess ? 0 : -EIO;
}

GFS_API int gfs_grep_graph_destroy(gfs_grep_graph* g) {
  if (!g) return -EINVAL;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(g->device);
  if (g->exec) cudaGraphExecDestroy(g->exec);
  if (g->d_str) cudaFree(g->d_str);
  cudaSetDevice(prev);
  delete g;
  return 0;
}
