// Host-side copy rates for the daemon's READ path: pread vs mmap+memcpy vs
// mmap + non-temporal stores, from a tmpfs file into per-thread page-size
// buffers, T threads. Usage: host_copy_bench FILE PAGE_KIB THREADS
#define _GNU_SOURCE
#include <fcntl.h>
#include <immintrin.h>
#include <pthread.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>
#include <sys/mman.h>
#include <sys/stat.h>
#include <time.h>
#include <unistd.h>

static const char* g_path;
static size_t g_page, g_size, g_npages;
static int g_threads, g_mode;
static const uint8_t* g_map;

static double now(void) {
  struct timespec ts;
  clock_gettime(CLOCK_MONOTONIC, &ts);
  return ts.tv_sec + ts.tv_nsec * 1e-9;
}

__attribute__((target("avx2"))) static void nt_copy(uint8_t* d, const uint8_t* s, size_t n) {
  size_t i = 0;
  for (; i + 128 <= n; i += 128) {
    __m256i a = _mm256_loadu_si256((const __m256i*)(s + i));
    __m256i b = _mm256_loadu_si256((const __m256i*)(s + i + 32));
    __m256i c = _mm256_loadu_si256((const __m256i*)(s + i + 64));
    __m256i e = _mm256_loadu_si256((const __m256i*)(s + i + 96));
    _mm256_stream_si256((__m256i*)(d + i), a);
    _mm256_stream_si256((__m256i*)(d + i + 32), b);
    _mm256_stream_si256((__m256i*)(d + i + 64), c);
    _mm256_stream_si256((__m256i*)(d + i + 96), e);
  }
  _mm_sfence();
  if (i < n) memcpy(d + i, s + i, n - i);
}

static void* worker(void* arg) {
  const int t = (int)(intptr_t)arg;
  uint8_t* buf = aligned_alloc(4096, g_page);
  mlock(buf, g_page);
  memset(buf, 0, g_page);
  int fd = open(g_path, O_RDONLY);
  for (size_t p = t; p < g_npages; p += g_threads) {
    const size_t off = p * g_page;
    if (g_mode == 0) {
      if (pread(fd, buf, g_page, off) < 0) abort();
    } else if (g_mode == 1) {
      memcpy(buf, g_map + off, g_page);
    } else {
      nt_copy(buf, g_map + off, g_page);
    }
  }
  close(fd);
  free(buf);
  return NULL;
}

int main(int argc, char** argv) {
  g_path = argv[1];
  g_page = (size_t)atoi(argv[2]) << 10;
  g_threads = atoi(argv[3]);
  struct stat st;
  stat(g_path, &st);
  g_size = st.st_size;
  g_npages = g_size / g_page;
  int fd = open(g_path, O_RDONLY);
  g_map = mmap(NULL, g_size, PROT_READ, MAP_SHARED, fd, 0);
  const char* names[3] = {"pread", "mmap+memcpy", "mmap+ntstore"};
  for (int rep = 0; rep < 2; ++rep) {
    for (g_mode = 0; g_mode < 3; ++g_mode) {
      pthread_t th[256];
      const double t0 = now();
      for (int i = 0; i < g_threads; ++i) pthread_create(&th[i], NULL, worker, (void*)(intptr_t)i);
      for (int i = 0; i < g_threads; ++i) pthread_join(th[i], NULL);
      const double dt = now() - t0;
      printf("%-14s threads=%d page=%zuKiB  %.2f GB/s\n", names[g_mode], g_threads, g_page >> 10,
             g_npages * g_page / dt / 1e9);
    }
  }
  return 0;
}
