/* gpufs_layout.h — memory layout shared by the host runtime (libgpufs.so) and
 * the header-only device library (gpufs_device.cuh). Plain C, no CUDA types.
 *
 * Everything here lives in one of three places (Fig. 2, §4):
 *   HBM (device memory)        — frame pool ("raw data array"),
 *                                per-frame metadata ("pframes"),
 *                                radix-tree node pool, open/closed
 *                                file table, RPC completion words;
 *   pinned, mapped host memory — the per-GPU RPC request queue;
 *   host only                  — daemon state (fd table, staging, streams).
 */
#ifndef GPUFS_LAYOUT_H
#define GPUFS_LAYOUT_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

/* ---- limits ---------------------------------------------------------- */
#define GFS_MAX_PATH 1024u     /* bytes incl. NUL; longer paths -> -ENAMETOOLONG */
#define GFS_FANOUT_SHIFT 8u    /* radix tree fanout 256 */
#define GFS_FANOUT (1u << GFS_FANOUT_SHIFT)
#define GFS_MAX_HEIGHT 4u      /* 256^4 = 2^32 pages per file */
#define GFS_MAX_BATCH 32u      /* pages looked up per warp-0 batch (one per lane) */
#define GFS_CTR_SHARDS 32      /* counters are sharded by SM id to avoid a hot address */

/* ---- open flags ------------------------------------------ */
#define GFS_O_RDONLY 0u
#define GFS_O_GWRONCE 1u       /* write-once, pages never fetched, pristine = zeros */
#define GFS_O_RDWR 2u          /* read-write with diff-and-merge write-back (NEXT-4):
                                  pages fetched from the host, a pristine copy kept per dirty page */
#define GFS_O_WRITABLE (GFS_O_GWRONCE | GFS_O_RDWR)
#define GFS_PROT_WRITE 2u      /* gmmap prot: the mapping will be written (O_RDWR files) */
#define GFS_O_PREFETCH 0x100u  /* gopen hint: fetch page 0 with the OPEN reply */

/* ---- config flags ------------------------------------------------------ */
#define GFS_F_LOCKED_TRAVERSAL 1u /* K5 ablation: every lookup takes the file lock */
#define GFS_F_NO_DMA_COMPLETION 2u /* fallback: completion via memcpy instead of stream write-value */
#define GFS_F_EXPORTED 4u          /* set by gfs_export: frames are published at system scope for peers */
#define GFS_F_NO_SPECULATE 8u      /* ablation: gread's one-page hits wait for the reference before copying */

/* ---- frame state word (pframe "state", 64 bits) -------------------------
 * bits 32..63 generation: +1 each time the frame is (re)assigned to a page.
 *             Leaf slots of the radix tree hold (generation << 32) | (frame+1),
 *             so one atomic increment both takes the reference and validates
 *             the slot (no separate tag load; install CAS cannot ABA).
 * bits 0..23  reference count (gread/gwrite copies and gmmap mappings)
 * bit  24     FILLING  — frame installed, contents not yet valid
 * bit  25     EVICTING — claimed by eviction / gfsync / truncate (ref was 0)
 * bit  26     ERROR    — fill failed; readers get -EIO
 */
#define GFS_ST_REF_MASK 0x00FFFFFFu
#define GFS_ST_FILLING (1u << 24)
#define GFS_ST_EVICTING (1u << 25)
#define GFS_ST_ERROR (1u << 26)
#define GFS_TAG_NONE 0xFFFFFFFFFFFFFFFFull /* tag = (uid << 32) | page index */
#define GFS_DIRTY_NONE 0xFFFFFFFFu
#define GFS_PRISTINE_PENDING 0xFFFFFFFFu
#define GFS_PF_POSTING 0xFFFFFFFFFFFFFFFFull /* f_pf: read-ahead frame installed, its RPC not posted yet */

/* ---- file table entry states (high byte of `sr`; low 24 bits = refcount) */
#define GFS_FS_FREE 0u
#define GFS_FS_CLAIM 1u
#define GFS_FS_OPENING 2u
#define GFS_FS_OPEN 3u
#define GFS_FS_CLOSED 4u
#define GFS_FS_REOPENING 5u
#define GFS_FS_DEAD 6u

typedef struct gfs_file {
  uint32_t sr;        /* (state << 24) | threadblock refcount */
  uint32_t uid;       /* cache incarnation id, never reused */
  uint32_t hfid;      /* daemon's host file id */
  uint32_t root;      /* radix root node index */
  uint64_t size;      /* size at first gopen / max written end */
  uint64_t version;   /* close-to-open version seen at (re)open */
  uint64_t ino, dev;
  int64_t mtime_ns;
  uint64_t path_hash;
  uint32_t path_len;
  uint32_t height;
  uint32_t oflags;
  uint32_t lock;      /* file spinlock for locked traversal */
  int32_t err;
  uint32_t pad;
  uint64_t synced_version; /* O_GWRONCE: host version after this cache's last write-back
                              (peer fill); 0 = none */
  uint64_t zc;             /* device address of the host file's registered page-cache mapping
                              (gfs_register_file; misses pull from it directly), 0 = none */
} gfs_file;

/* ---- RPC (§4.3) -------------------------------------------- */
#define GFS_OP_NOP 0u
#define GFS_OP_OPEN 1u     /* path -> hfid, size, version, ino, dev, mtime */
#define GFS_OP_READ 2u     /* pread(hfid, len, off) -> DMA to dev_ptr */
#define GFS_OP_WRITE 3u    /* DMA from dev_ptr -> pwrite(hfid, len, off), version++ */
#define GFS_OP_CLOSE 4u    /* close(hfid) */
#define GFS_OP_TRUNC 5u    /* ftruncate(hfid, arg) */

#define GFS_WF_FULL 1u     /* WRITE: every byte of [off,off+len) was written (no merge) */
#define GFS_WF_DIFF 2u     /* WRITE (O_RDWR): write only the bytes where staging slot `stage` (working
                              copy) differs from staging slot `arg` (pristine copy) */
#define GFS_WF_MASK 4u     /* WRITE (O_RDWR): staging slot `arg` holds a bitmap over [off, off+len)
                              (64-bit words, bit j of word w = byte 64w + j; off is 64-aligned in the
                              page): write only the marked bytes of slot `stage` */

typedef struct gfs_rpc_req { /* one 64-byte ring slot in pinned host memory */
  uint32_t op;
  uint32_t hfid;
  uint64_t file_off;
  uint64_t dev_ptr;
  uint32_t len;
  uint32_t flags;
  uint64_t arg;
  uint32_t path_len;
  uint32_t stage;    /* READ/WRITE: staging slot holding the data (host-mapped pinned memory) */
  uint64_t pad1;
  uint64_t seq;      /* = ticket + 1; written LAST with st.release.sys */
} gfs_rpc_req;

typedef struct gfs_rpc_resp { /* OPEN reply, host-written before completion */
  int64_t size;
  uint64_t version;
  uint64_t ino, dev;
  int64_t mtime_ns;
  uint32_t hfid;
  int32_t status;
  uint64_t pad[2];
} gfs_rpc_resp;

/* completion word (pinned, mapped host memory; host store-release, GPU
 * ld.acquire.sys): ((ticket + 1) << 32) | (uint32_t)result. The daemon makes
 * no CUDA call per RPC: data moves through host-mapped staging slots that the
 * GPU itself reads (fill) or writes (write-back) over PCIe. */

/* ---- counters (Table 2 analogue + RPC accounting) --------------------- */
enum {
  GFS_C_HIT = 0,        /* page found valid, lock-free */
  GFS_C_MISS,           /* page installed and fetched from host */
  GFS_C_ZERO_FILL,      /* O_GWRONCE page installed zero-filled */
  GFS_C_LOCKFREE,       /* lookups that succeeded without the lock */
  GFS_C_LOCKED,         /* lookups that took the file lock (incl. retries) */
  GFS_C_RETRY,          /* optimistic validation failures */
  GFS_C_EVICT,          /* frames reclaimed */
  GFS_C_WRITEBACK,      /* dirty ranges written back */
  GFS_C_RPC,            /* RPCs posted */
  GFS_C_RPC_OPEN,
  GFS_C_RPC_READ,
  GFS_C_RPC_WRITE,
  GFS_C_BYTES_H2D,
  GFS_C_BYTES_D2H,
  GFS_C_OPEN_FAST,      /* gopen served without RPC */
  GFS_C_REOPEN_VALID,   /* closed-file cache revalidated and kept */
  GFS_C_INVALIDATE,     /* closed-file cache dropped on re-open */
  GFS_C_ENOMEM,
  GFS_C_TIMEOUT,
  GFS_C_GREAD_CALLS,
  GFS_C_GREAD_BYTES,
  GFS_C_GWRITE_CALLS,
  GFS_C_NODES,          /* radix nodes allocated */
  GFS_C_RING_WAIT,      /* ring slot was busy on post */
  GFS_C_BUSY,           /* lookups that found the page being filled/evicted by another block */
  GFS_C_STAGE_WAIT,     /* staging slot allocation had to wait */
  GFS_C_PEER_FILL,      /* misses filled from a peer GPU's cache (NVLink) instead of the host */
  GFS_C_BYTES_PEER,     /* bytes copied from peer caches */
  GFS_C_PEER_MISS,      /* misses for which no peer held a usable copy */
  GFS_C_ZC_FILL,        /* misses filled straight from a registered file mapping (no RPC) */
  GFS_C_RA_ISSUED,      /* read-ahead fetches posted (NEXT-2) */
  GFS_C_RA_ADOPTED,     /* read-ahead fills completed by a lookup that needed the page */
  GFS_C_RA_REAPED,      /* read-ahead fills completed by their issuer's gclose (page not read meanwhile) */
  GFS_C_NCOUNTERS
};

/* ---- peer caches (NEXT-1: the buffer cache spans GPUs)
 * A read-only view of another GPU's cache, every pointer valid in THIS
 * process's address space (CUDA IPC mapping, or the exporter's own pointers
 * when both caches live in one process). A miss may be filled from a peer
 * frame over NVLink instead of the host; see gpufs_device.cuh peer_take. */
#define GFS_MAX_PEERS 8u
typedef struct gfs_peer {
  uint8_t* pool;
  uint64_t* f_state;
  uint64_t* f_tag;
  uint32_t* f_lo;
  uint32_t* f_hv;
  uint64_t* nodes;
  gfs_file* files;
  uint32_t nframes, max_nodes, max_files, page_shift;
} gfs_peer;

/* ---- the device context (lives in HBM; kernels receive a pointer) ------ */
typedef struct gfs_ctx {
  uint64_t page_size;
  uint32_t page_shift;
  uint32_t nframes;
  uint8_t* pool;
  /* pframes, SoA */
  uint64_t* f_state;  /* generation << 32 | flags | refcount */
  uint64_t* f_tag;
  uint32_t* f_file;
  uint32_t* f_valid;
  uint32_t* f_lo;
  uint32_t* f_hi;
  uint32_t* f_written;
  uint32_t* f_stamp;
  uint32_t* f_hv;     /* bytes [0, hv) equal the host file at the entry's version (peer fill) */
  uint32_t* f_pristine; /* O_RDWR dirty page: pristine frame + 1 (0 none, GFS_PRISTINE_PENDING being made) */
  uint32_t* fresh_next;
  uint32_t* hand;
  /* radix node pool: 64-bit entries (interior: child node id; leaf: gen << 32 | frame + 1) */
  uint64_t* nodes;
  uint32_t max_nodes;
  uint32_t max_files; /* power of two */
  uint32_t* node_next;
  uint32_t* node_free;
  uint32_t* node_free_top;
  uint32_t* node_lock;
  /* file table */
  gfs_file* files;
  char* paths;
  uint32_t* uid_next;
  uint32_t ring_slots;
  /* RPC */
  gfs_rpc_req* ring;   /* device-mapped pointer to pinned host ring */
  gfs_rpc_resp* resp;  /* device-mapped pointer to pinned host responses */
  char* ring_paths;    /* device-mapped, ring_slots * GFS_MAX_PATH */
  uint64_t* cpl;       /* device-mapped pinned host memory: completion words */
  uint64_t* ack;       /* device memory: slot released by its client */
  unsigned long long* ring_tail;
  /* staging: pinned host slots of page_size bytes, device-mapped */
  uint8_t* staging;
  uint32_t staging_slots;
  uint32_t staging_words;  /* bitmap words */
  uint32_t* staging_bits;  /* device memory: 1 = slot in use */
  uint32_t pad_staging;
  /* config */
  uint32_t flags;
  uint32_t max_batch;
  uint64_t timeout_ns;
  unsigned long long* ctr;
  /* peer caches (device array of npeers views) */
  const gfs_peer* peers;
  uint32_t npeers;
  uint32_t readahead;  /* pages fetched ahead of a block's sequential gread of a read-only file (0 = off) */
  /* read-ahead (NEXT-2): per frame, a fill in flight that no reader waits for yet:
   * 0 none, GFS_PF_POSTING being posted, else ((ticket + 1) << 32) | (staging slot + 1) */
  uint64_t* f_pf;
} gfs_ctx;

#ifdef __cplusplus
}
#endif
#endif /* GPUFS_LAYOUT_H */
