/* gpufs.h — host-side C ABI of libgpufs.so (the B200 GPUfs buffer-cache read path).
 *
 * extern "C", plain pointers and sizes only (no torch / CUDA runtime types in
 * signatures: streams are passed as `void*` holding a cudaStream_t / CUstream,
 * device buffers as plain pointers). Every call returns 0 or a positive value
 * on success and -errno on failure.
 *
 * Layers (Fig. 2):
 *   - gfs_init / gfs_shutdown: allocate / free the GPU buffer cache (raw data
 *     array P:L595-596, pframes P:L597-606, radix-tree nodes P:L612-622, file
 *     tables) and the per-GPU RPC queue in pinned memory.
 *   - gfs_daemon / gfs_daemon_stop: the host side of the GPU->CPU RPC
 *     (P:L675-740): worker threads poll the queue, pread into pinned staging
 *     and DMA into cache frames, write back dirty ranges, keep a
 *     close-to-open version table (user-space stand-in for WRAPFS).
 *   - gfs_run_*: launchers of the kernels built on the device API
 *     (include/gpufs_device.cuh). They enqueue on `stream` and return without
 *     synchronising. The daemon must be running while they execute.
 *
 * Ownership: the library owns everything it allocates (unless
 * gfs_config.frame_pool supplies caller-owned device memory for the frames).
 * Device buffers passed to gfs_run_* are owned by the caller and must stay
 * valid until the stream reaches the launch. Not thread-safe: call the host
 * API from one thread per handle.
 */
#ifndef GPUFS_H
#define GPUFS_H

#include <stdint.h>
#include "gpufs_layout.h"

#ifdef __cplusplus
extern "C" {
#endif

typedef struct gfs_config {
  int device;               /* CUDA ordinal */
  uint64_t cache_bytes;     /* frame pool bytes (paper: 2 GB) */
  uint32_t page_size;       /* power of two, 4 KiB .. 16 MiB (configurable) */
  uint32_t ring_slots;      /* RPC queue entries (power of two) */
  uint32_t daemon_threads;  /* host worker threads (pread + DMA channels) */
  uint32_t max_files;       /* open+closed file table entries (power of two) */
  uint32_t max_nodes;       /* radix node pool (0 = auto) */
  uint32_t max_batch;       /* pages looked up per warp-0 batch, 1..32 */
  uint32_t flags;           /* GFS_F_* (gpufs_layout.h) */
  uint32_t staging_slots;   /* pinned host staging slots of page_size bytes (0 = auto: 128 MiB worth) */
  uint64_t timeout_ms;      /* device-side wait bound (0 = none) -> -ETIMEDOUT */
  void* frame_pool;         /* optional caller-owned device memory >= cache_bytes */
  uint32_t readahead;       /* NEXT-2: pages a block's sequential gread of a read-only file fetches ahead
                               (READ RPCs posted, not waited for), 0 = off, at most 8 */
  uint32_t fault;           /* tests: daemon fault injection, GFS_FAULT_* kind << 24 | period (0 = off) */
} gfs_config;

/* Daemon fault injection (tests): every `period`-th READ RPC of a
 * file of at least 2 pages fails with -EIO (GFS_FAULT_EIO) or returns half the
 * bytes it was asked for (GFS_FAULT_SHORT; the GPU zero-fills the rest, as
 * for a file that shrank under the cache, R4). */
#define GFS_FAULT_EIO 1u
#define GFS_FAULT_SHORT 2u

typedef struct gfs_handle gfs_handle;

#define GFS_DAEMON_SPAWN 0  /* start worker threads and return */
#define GFS_DAEMON_RUN 1    /* start workers, block the caller until gfs_daemon_stop */

/* Fill *cfg with defaults (64 KiB pages, 1 GiB cache, 4096 slots, 8 threads). */
int gfs_config_default(gfs_config* cfg);

/* Allocate the cache and the RPC channel on cfg->device. No kernel may use
 * the context before this returns. -EINVAL on bad geometry, -ENOMEM on
 * allocation failure, -ENODEV if CUDA is unavailable. */
int gfs_init(const gfs_config* cfg, gfs_handle** out);

/* Start the host daemon (mode GFS_DAEMON_SPAWN / GFS_DAEMON_RUN). Uses only
 * non-blocking streams and never synchronises the device. */
int gfs_daemon(gfs_handle* h, int mode);

/* Stop the daemon threads (in-flight RPCs are finished first). */
int gfs_daemon_stop(gfs_handle* h);

/* Free everything. Dirty pages are NOT flushed (gclose != sync). */
int gfs_shutdown(gfs_handle* h);

/* Device pointer to the gfs_ctx to pass to kernels using gpufs_device.cuh. */
const gfs_ctx* gfs_device_ctx(gfs_handle* h);

/* ---- peer caches (NEXT-1; the cache "spans multiple GPUs", P:L136-137,
 * P:L452-454). Each GPU keeps its own cache (one process per GPU);
 * a cache that attaches its peers fills an O_RDONLY miss from a peer frame
 * over NVLink when the peer holds the same host file at the same
 * close-to-open version, clean and host-verified, and asks
 * the host otherwise. Results are identical either way. */
typedef struct gfs_export_desc {
  uint64_t magic;
  int32_t pid, device;
  uint32_t page_shift, nframes, max_nodes, max_files;
  uint64_t ptr[7];              /* exporter's device pointers (same-process attach) */
  unsigned char ipc[7][64];     /* cudaIpcMemHandle_t of: pool, f_state, f_tag, f_lo, f_hv, nodes, files */
} gfs_export_desc;

/* Describe this cache for gfs_attach_peer in another process (or handle) and
 * switch its fills to system-scope publication. Plain bytes: send them to
 * the peer with any transport (e.g. torch.distributed all_gather_object).
 * Call before any kernel uses the context. -ENOTSUP if the frame pool is
 * caller-owned (gfs_config.frame_pool), -EIO if CUDA IPC is unavailable. */
int gfs_export(gfs_handle* h, gfs_export_desc* out);

/* Map the cache described by `d` (CUDA IPC across processes, direct pointers
 * within one process, peer access enabled across devices) as a read-only
 * peer of h. Returns the peer index (>= 0). Same page size required
 * (-EINVAL); at most GFS_MAX_PEERS (-ENOSPC); -EIO if the mapping fails.
 * No kernel may use h's context during the call. The exporter must outlive
 * every kernel of h that runs after the attach (shut h down first, or
 * barrier). */
int gfs_attach_peer(gfs_handle* h, const gfs_export_desc* d);

/* Zero-copy misses: map `path` (an existing, non-empty file) into the GPU's
 * address space with cudaHostRegister: first a read-only shared mapping
 * registered read-only (cudaHostRegisterReadOnly: the file may be read-only to
 * the caller, and no device store can reach it); if the driver refuses that,
 * a read-write shared mapping. Later O_RDONLY opens of the same file (same
 * st_dev, st_ino and size) fill their misses by pulling the page straight
 * from the host page cache over PCIe: no READ RPC, no staging slot, no daemon
 * memcpy. A setup call (seconds per tens of GiB); the mapping lives until
 * gfs_shutdown. The file must not change size or be replaced while
 * registered (weak consistency as for any open file, R4). Returns 1 (read-only
 * registration) or 0 (read-write), -errno on failure (-EIO if CUDA refuses
 * the registration). */
int gfs_register_file(gfs_handle* h, const char* path);

/* Copy the device counters (GFS_C_*, summed over shards) into out[0..n). */
int gfs_stats(gfs_handle* h, uint64_t* out, int n, int reset);

/* Host daemon counters: out[0..n): rpcs, reads, writes, opens, closes, truncs,
 * bytes_h2d, bytes_d2h, pread_ns, errors, merges. */
int gfs_host_stats(gfs_handle* h, uint64_t* out, int n);

/* Geometry: out[0]=page_size out[1]=nframes out[2]=max_files out[3]=max_nodes
 * out[4]=ring_slots out[5]=daemon_threads out[6]=stream-write-value-64 used. */
int gfs_info(gfs_handle* h, uint64_t* out, int n);

/* --------------------------------------------------------------------------
 * Kernel launchers (device-side calls run inside these kernels).
 * `path` arguments are host NUL-terminated strings; the launcher stages them in
 * device memory. All d_* pointers are device memory. grid/block: launch shape.
 * Return 0 once enqueued, -EINVAL on bad arguments, or a CUDA error as -EIO.
 * ------------------------------------------------------------------------ */

/* Parity harness: each block gopen()s `path` (flags), then issues calls
 * i = blockIdx.x, blockIdx.x + grid, ... < ncalls:
 *   mode 0: d_ret[i] = gread(fd, d_off[i], d_len[i], d_dst + d_dstoff[i])
 *   mode 1: p = gmmap(.., d_len[i], .., fd, d_off[i], &m); copy m bytes to
 *           d_dst + d_dstoff[i]; gmunmap; d_ret[i] = p ? m : -errno-or-0
 *   mode 2: like mode 0 but the destination is dynamic shared memory
 *           (requires d_len[i] <= smem_bytes), copied out to d_dst afterwards
 *   mode 3: like mode 2 with the destination at smem + d_off[i] % 16, i.e.
 *           co-aligned with the file offset (requires d_len[i] + 15 <= smem_bytes)
 * then gclose().
 *   mode 4: warp-collective calls instead (gopen_warp / gread_warp /
 *           gclose_warp): warp w of the grid issues calls w, w + nwarps, ...
 *           into global memory. block: a multiple of 32, at most
 *           32 * GFS_WARP_API_MAX_WARPS (256).
 *   mode 5: like mode 4 into the warp's own shared buffer of smem_bytes
 *           (co-aligned at d_off[i] % 16), copied out afterwards. If gopen fails every d_ret[i] of that block gets its error.
 * Bits 8+ of mode: the open flags of modes 0-3 (GFS_O_RDONLY, or GFS_O_RDWR to read
 * a file the GPU also writes); modes 4-5 open read-only. */
int gfs_run_gread(gfs_handle* h, void* stream, const char* path, int mode, uint32_t ncalls,
                  const uint64_t* d_off, const uint64_t* d_len, const uint64_t* d_dstoff, uint8_t* d_dst,
                  int64_t* d_ret, uint32_t grid, uint32_t block, uint32_t smem_bytes);

/* Sequential sweep (C2 / K1 shape): block b reads its contiguous
 * range of [file_off, file_off + total) in `chunk`-byte calls — gread into
 * d_scratch + b*chunk (use_mmap = 0) or gmmap (use_mmap = 1) — and adds the
 * position-weighted checksum sum_j w_j*(2j+1) of the bytes read (j = global
 * 8-byte word index) into *d_sum. use_mmap = 2: gread only, into
 * d_scratch + (o - file_off) (a destination of `total` bytes: the cache-hit
 * gread -> global measurement; *d_sum untouched). Ranges are split in
 * multiples of chunk. *d_err receives the most negative error seen (0 if none). */
int gfs_run_seqread(gfs_handle* h, void* stream, const char* path, uint64_t file_off, uint64_t total,
                    uint64_t chunk, int use_mmap, uint8_t* d_scratch, uint64_t* d_sum, int64_t* d_err,
                    uint32_t grid, uint32_t block);

/* Cache-hit read benchmark (K4 shape): block b issues
 * calls_per_block greads of `chunk` bytes into dynamic shared memory at file
 * offsets d_off[b*calls_per_block + i] (chunk-aligned), checksumming each
 * chunk from shared memory into *d_sum. raw: 0 = gread; 1 = the baseline: the
 * same copies straight from d_raw (the file's bytes already in device memory),
 * without GPUfs (h may be NULL then); 2 = gread_hint, each call naming the
 * block's next offset (split-phase lookup: the next page is looked up and
 * referenced while the current copy is in flight). */
int gfs_run_randread(gfs_handle* h, void* stream, const char* path, int raw, const uint8_t* d_raw,
                     uint32_t chunk, uint32_t calls_per_block, const uint64_t* d_off, uint64_t* d_sum,
                     int64_t* d_err, uint32_t grid, uint32_t block);

/* Host->device link probe (the miss path's roofline): best of `reps` over
 * nbytes (>= 1 MiB, multiple of 16) of mapped pinned host memory, moved (a) by
 * the copy engine (cudaMemcpyAsync) into *ce_gbps and (b) by SMs pulling
 * 16-byte words (__ldcv, as gread pulls staging slots) into *sm_gbps, in
 * GB/s (1e9 B/s). Allocates and frees its own buffers; synchronises `stream`.
 * -EINVAL on bad arguments, -ENOMEM if the buffers cannot be allocated. */
int gfs_probe_h2d(void* stream, uint64_t nbytes, uint32_t reps, double* ce_gbps, double* sm_gbps);

/* The same benchmark with the warp-collective API (gread_warp):
 * block/32 warps per block, each with its own `chunk` bytes of shared memory,
 * warp w of block b issuing calls w, w + block/32, ... of block b's
 * calls_per_block. block: a multiple of 32, at most 256. */
int gfs_run_randread_warp(gfs_handle* h, void* stream, const char* path, int raw, const uint8_t* d_raw,
                          uint32_t chunk, uint32_t calls_per_block, const uint64_t* d_off, uint64_t* d_sum,
                          int64_t* d_err, uint32_t grid, uint32_t block);

/* The same benchmark with the split-phase lane-parallel gread (NEXT-2,
 * gread_lanes_issue / gread_lanes_wait): warp 0 of each block issues the next
 * `depth` calls (one lane each) into one half of a double buffer of
 * 2 * depth * chunk bytes of shared memory while the block checksums the other
 * half. raw: the same schedule with plain TMA copies from d_raw. block: a
 * multiple of 32, <= 256; depth <= 32; 2 * depth * chunk <= 200 KiB. */
int gfs_run_randread_async(gfs_handle* h, void* stream, const char* path, int raw, const uint8_t* d_raw,
                           uint32_t chunk, uint32_t calls_per_block, uint32_t depth, const uint64_t* d_off,
                           uint64_t* d_sum, int64_t* d_err, uint32_t grid, uint32_t block);

/* Write harness: each block gopen(path, flags) — GFS_O_GWRONCE (write-once,
 * diff against zeros) or GFS_O_RDWR (pages fetched, diff against
 * a pristine copy) — and issues
 * d_ret[i] = gwrite(fd, d_off[i], d_len[i], d_src + d_srcoff[i]) for its calls,
 * then gclose. -EINVAL for other flags. */
int gfs_run_gwrite(gfs_handle* h, void* stream, const char* path, uint32_t ncalls, const uint64_t* d_off,
                   const uint64_t* d_len, const uint64_t* d_srcoff, const uint8_t* d_src, int64_t* d_ret,
                   uint32_t grid, uint32_t block, int flags);

/* Writable-mapping harness (O_RDWR, Tab.1 gmmap/gmsync): block b
 * takes calls b, b + grid, ...: gmmap(d_off[i], d_len[i], GFS_PROT_WRITE), store
 * d_src + d_srcoff[i] through the pointer (the mapped prefix only), gmsync the
 * page if do_msync, gmunmap. d_ret[i] = bytes mapped or -errno. */
int gfs_run_mmap_write(gfs_handle* h, void* stream, const char* path, uint32_t ncalls, const uint64_t* d_off,
                       const uint64_t* d_len, const uint64_t* d_srcoff, const uint8_t* d_src, int64_t* d_ret,
                       uint32_t grid, uint32_t block, int do_msync);

/* One-block file operations: op 0 = gfsync, 1 = gftruncate(arg), 2 = gfstat_size,
 * 3 = gopen+gclose only, 4 = pin (gopen without gclose: the file stays open
 * across launches, *d_ret = fd), 5 = unpin (gclose(fd = arg)), 6 = gfsync from `arg`
 * blocks at once (they split the dirty pages by claim) followed by a strict
 * one-block pass; *d_ret = 0 or the most negative error.
 * flags = open flags. *d_ret = result. */
/* C5 write side: pin `path` open O_GWRONCE (one
 * reference held for the duration), then `grid` blocks gwrite() [0, total)
 * from device buffer d_src in `chunk`-byte calls (block b takes a contiguous
 * share), then `sync_grid` blocks call gfsync() on it concurrently (dirty pages
 * are claimed by CAS, so they split the write-back; -EBUSY from a page another
 * of them holds is expected) followed, when sync_grid > 1, by one strict
 * single-block gfsync that must find every page clean, then the pin is dropped
 * (gclose, no write-back). All on `stream`. *d_err: 0 or the most negative
 * error (caller zeroes it); d_tmp: one device int64 of scratch (pinned fd).
 * sync_grid * min(32, block) must not exceed the staging slots (each writing
 * lane holds one while it waits for its RPC). */
int gfs_run_seqwrite(gfs_handle* h, void* stream, const char* path, uint64_t total, uint64_t chunk,
                     const uint8_t* d_src, int64_t* d_err, int64_t* d_tmp, uint32_t grid, uint32_t block,
                     uint32_t sync_grid);

int gfs_run_fileop(gfs_handle* h, void* stream, const char* path, int flags, int op, uint64_t arg,
                   int64_t* d_ret);

/* --------------------------------------------------------------------------
 * grep -w consumer (§5.2.2): for each word of the dictionary
 * (one word per 32-byte slot) count how many times and in which
 * files it appears; the input file names are read from the
 * list file (one path per line, relative to the list's directory,
 * P:L1266-1267). Word bytes are [A-Za-z0-9_]; counts are per occurrence.
 * ------------------------------------------------------------------------ */
typedef struct gfs_grep_params {
  uint32_t max_files;   /* capacity of the file list */
  uint32_t max_words;   /* capacity of the dictionary (words) */
  uint64_t list_cap;    /* bytes of the list file (capacity) */
  uint64_t pair_cap;    /* (file, word) table slots (rounded up to a power of two) */
  uint64_t hit_cap;     /* hits to list in d_hits (0: none) */
  uint32_t chunk;       /* work-item bytes: a file larger than this is split into chunks of it;
                           multiple of 16, at most 65472 (item + halos < 64 KiB: 16-bit offsets) */
  uint32_t grid;        /* persistent blocks (at most one per resident block slot) */
  uint32_t block;       /* threads per block, multiple of 32, <= 256 */
  uint32_t keep_open;   /* 1: leave every file (and the dictionary and list) open after the run:
                           warm re-runs skip the host (no close-to-open revalidation) */
  uint64_t corpus_cap;  /* bytes of all listed files (capacity, sizes the work-item map) */
  const uint32_t* file_ids; /* device array: file i of the list is reported as file_ids[i] in
                           records, hits and the digest (e.g. a shard's global indices); NULL:
                           the list index i */
  uint64_t rec_cap;     /* records the work area can stage (>= the records found, else -ENOSPC) */
  uint32_t whole_max;   /* a file of more than one chunk and at most this many bytes is ONE work
                           item: one block scans it chunk after chunk, counting in shared memory,
                           and emits its records directly (0: 64 bytes per count-table slot, the
                           slots being what shared memory allows at >= 768 threads per SM:
                           4096 at block 256 / chunk 16 KiB, 1024 at block 128; <= chunk: never). Larger
                           files are split into chunk items merged through the (file, word) table */
  uint32_t scan;        /* 0: block scan (one block per item, items staged in shared memory by
                           gread/TMA); 1: warp scan (one warp per item, no block barrier, the
                           text read in place through gmmap_warp; needs chunk a multiple of 1024
                           and <= 65536, whole_max <= 65536, max_words < 65535) */
} gfs_grep_params;

/* Device scratch bytes gfs_grep needs for these parameters. */
uint64_t gfs_grep_work_bytes(const gfs_grep_params* p);

/* Enqueue the whole search on `stream`. Outputs (device memory, caller-owned):
 *   d_rec[3*i .. 3*i+2] = (file index, word index, count), unique pairs, unordered,
 *                         up to rec_cap records (d_summary[0] = records found);
 *   d_totals[k]         = occurrences of word k over all files (max_words entries);
 *   d_hits[2*i], [2*i+1] = ((file << 32) | word, byte offset) per hit if non-NULL,
 *                         up to hit_cap (d_summary[8] = hits listed + dropped);
 *   d_summary[0..9]     = nrecords, nhits, digest_sum, digest_xor, nfiles, nwords,
 *                         corpus bytes, error (0 or -errno), nhits_listed, nitems.
 * The digest is sum and xor over hits of splitmix64(splitmix64(splitmix64(f)+off)+k)
 * (order independent). File index = position among the list's non-empty lines, or
 * file_ids[position] when given. The work area also carries state across runs
 * with the same d_work (an empty (file, word) table, the held dictionary and
 * list with keep_open): reuse it only with the same parameters. */
int gfs_grep(gfs_handle* h, void* stream, const char* dict_path, const char* list_path,
             const gfs_grep_params* p, void* d_work, uint32_t* d_rec, uint64_t rec_cap, uint64_t* d_totals,
             uint64_t* d_hits, uint64_t* d_summary);

/* The same grep run captured once as a CUDA graph and replayed (the pipeline
 * is ~16 small kernels: launch-bound for small corpora). gfs_grep_graph_create
 * captures exactly what gfs_grep would enqueue for these arguments (the path
 * strings are copied into device memory the graph owns; parameters, buffers and
 * the cache context are fixed at capture: re-create the graph after gfs_export /
 * gfs_attach_peer or to change any argument); `stream` is unused (capture runs
 * on a private stream; nothing executes). gfs_grep_graph_launch enqueues one
 * run on `stream`: the same results and work-area state as gfs_grep.
 * Returns 0 or -errno (-EINVAL bad arguments, -ENAMETOOLONG a path,
 * -EIO capture or instantiation failed). */
typedef struct gfs_grep_graph gfs_grep_graph;
int gfs_grep_graph_create(gfs_handle* h, void* stream, const char* dict_path, const char* list_path,
                          const gfs_grep_params* p, void* d_work, uint32_t* d_rec, uint64_t rec_cap,
                          uint64_t* d_totals, uint64_t* d_hits, uint64_t* d_summary, gfs_grep_graph** out);
int gfs_grep_graph_launch(gfs_grep_graph* g, void* stream);
int gfs_grep_graph_destroy(gfs_grep_graph* g);

/* --------------------------------------------------------------------------
 * Out-of-core fp32 matrix-vector product (§5.1.4): y = A x with
 * A a row-major little-endian fp32 file (rows x cols), x a cols-long fp32
 * file, y written to y_path through gftruncate + gwrite + gfsync (O_GWRONCE).
 * A is consumed through gmmap page by page; products accumulate in fp64 and
 * each y_r is rounded to fp32 once. d_x: device scratch of cols floats (x is
 * gread into it). d_y: optional device copy of y (rows floats). *d_err:
 * 0 or the most negative error. Needs ceil(rows/grid)*4 <= 160 KiB (y slice
 * of a block in shared memory).
 * ------------------------------------------------------------------------ */
int gfs_matvec(gfs_handle* h, void* stream, const char* a_path, const char* x_path, const char* y_path,
               uint64_t rows, uint64_t cols, float* d_x, float* d_y, int64_t* d_err, uint32_t grid,
               uint32_t block);

/* The same for the row block [row0, row0 + nrows) of A (a rank's shard in the
 * multi-GPU C3): y_path and d_y receive those nrows values only
 * (y_path's element i is y_{row0+i}). -EINVAL if the range is empty or
 * exceeds rows. */
int gfs_matvec_rows(gfs_handle* h, void* stream, const char* a_path, const char* x_path, const char* y_path,
                    uint64_t rows, uint64_t cols, uint64_t row0, uint64_t nrows, float* d_x, float* d_y,
                    int64_t* d_err, uint32_t grid, uint32_t block);

#ifdef __cplusplus
}
#endif
#endif /* GPUFS_H */
