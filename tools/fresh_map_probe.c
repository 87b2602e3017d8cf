// Host copy rates of a FRESHLY WRITTEN tmpfs file (the C5 re-read case) into
// per-thread 2 MiB buffers, T threads, regions interleaved by thread:
//   fresh : first memcpy through a new PROT_READ mapping (page-table faults)
//   warm  : the same mapping again (populated)
//   pread : pread_full
//   popul : a new mapping, madvise(MADV_POPULATE_READ) per region, then memcpy
// Usage: fresh_map_probe FILE MIB THREADS
#define _GNU_SOURCE
#include <fcntl.h>
#include <pthread.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>
#include <sys/mman.h>
#include <time.h>
#include <unistd.h>
#ifndef MADV_POPULATE_READ
#define MADV_POPULATE_READ 22
#endif
static size_t g_size, g_reg = 2 << 20;
static int g_threads, g_mode, g_fd;
static const uint8_t* g_map;
static double now(void) {
  struct timespec ts;
  clock_gettime(CLOCK_MONOTONIC, &ts);
  return ts.tv_sec + ts.tv_nsec * 1e-9;
}
static void* worker(void* arg) {
  const long t = (long)arg;
  uint8_t* buf = aligned_alloc(4096, g_reg);
  memset(buf, 0, g_reg);
  for (size_t r = t; r * g_reg < g_size; r += g_threads) {
    const size_t off = r * g_reg;
    if (g_mode == 2) {
      size_t done = 0;
      while (done < g_reg) {
        ssize_t n = pread(g_fd, buf + done, g_reg - done, off + done);
        if (n <= 0) break;
        done += n;
      }
    } else {
      if (g_mode == 3 && madvise((void*)(g_map + off), g_reg, MADV_POPULATE_READ) != 0) perror("madvise");
      memcpy(buf, g_map + off, g_reg);
    }
  }
  free(buf);
  return NULL;
}
static double run(int mode) {
  g_mode = mode;
  pthread_t th[64];
  const double t0 = now();
  for (long i = 0; i < g_threads; ++i) pthread_create(&th[i], NULL, worker, (void*)i);
  for (int i = 0; i < g_threads; ++i) pthread_join(th[i], NULL);
  return g_size / (now() - t0) / 1e9;
}
static void write_file(const char* p, int seed) {
  int fd = open(p, O_CREAT | O_TRUNC | O_RDWR, 0644);
  uint8_t* b = malloc(g_reg);
  for (size_t o = 0; o < g_size; o += g_reg) {
    memset(b, (int)(o >> 21) + seed, g_reg);
    if (pwrite(fd, b, g_reg, o) != (ssize_t)g_reg) perror("pwrite");
  }
  free(b);
  close(fd);
}
int main(int argc, char** argv) {
  const char* path = argv[1];
  g_size = (size_t)atol(argv[2]) << 20;
  g_threads = atoi(argv[3]);
  for (int it = 0; it < 2; ++it) {
    write_file(path, it);
    g_fd = open(path, O_RDONLY);
    g_map = mmap(NULL, g_size, PROT_READ, MAP_SHARED, g_fd, 0);
    const double fresh = run(0), warm = run(1), pr = run(2);
    munmap((void*)g_map, g_size);
    g_map = mmap(NULL, g_size, PROT_READ, MAP_SHARED, g_fd, 0);
    const double pop = run(3);
    munmap((void*)g_map, g_size);
    close(g_fd);
    printf("iter %d, %zu MiB, %d threads: fresh mmap %.1f GB/s, warm mmap %.1f, pread %.1f, populate+memcpy %.1f\n", it,
           g_size >> 20, g_threads, fresh, warm, pr, pop);
  }
  unlink(path);
  return 0;
}
