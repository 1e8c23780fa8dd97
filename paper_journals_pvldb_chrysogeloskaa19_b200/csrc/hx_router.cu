// hx_router.cu — the router's dynamic load balancing across processes (§8(e) host-resident;
// §8(a) a2, a8).
//
// PAPER.md:469-473 §3.1: the router "routes partitions to consumers, while load-balancing";
// with a dynamic policy a block goes to whichever consumer asks for work first. One process
// per GPU means the consumers do not share an address space, so the block counter lives in
// POSIX shared memory: every process of the node opens the same segment and draws block
// indices with an atomic fetch-add. The blocks themselves are the row ranges of a
// host-resident (pinned) fact table that every process maps (the SF1000
// data stays in CPU memory and is streamed to the GPUs); a GPU draws its next block only when
// a slot of its staging ring is free, so a faster GPU (or link) simply draws more blocks.
#include <fcntl.h>
#include <sys/mman.h>
#include <sys/stat.h>
#include <unistd.h>

#include <atomic>
#include <cstring>
#include <string>

#include "hx_internal.cuh"

namespace {
struct SharedCounter {
  std::atomic<int64_t> next;
  int64_t n_blocks;
  int64_t magic;
};
constexpr int64_t kMagic = 0x6878726f75746572LL;  // "hxrouter"
static_assert(std::atomic<int64_t>::is_always_lock_free, "lock-free 64-bit atomic in shared memory");
}  // namespace

struct hx_shared_router {
  std::string name;
  int fd = -1;
  SharedCounter* c = nullptr;
};

using namespace hx;

extern "C" {

int hx_shared_router_open(const char* name, int64_t n_blocks, int create, hx_shared_router** out) {
  HX_REQUIRE(name && name[0] == '/' && std::strchr(name + 1, '/') == nullptr && out && n_blocks >= 0,
             HX_EINVAL, "hx_shared_router_open: name must be \"/word\", n_blocks >= 0");
  const int fd = shm_open(name, create ? (O_CREAT | O_RDWR) : O_RDWR, 0600);
  HX_REQUIRE(fd >= 0, HX_EINVAL, std::string("hx_shared_router_open: shm_open: ") + std::strerror(errno));
  if (create && ftruncate(fd, sizeof(SharedCounter)) != 0) {
    close(fd);
    return fail(HX_ENOMEM, "hx_shared_router_open: ftruncate failed");
  }
  void* p = mmap(nullptr, sizeof(SharedCounter), PROT_READ | PROT_WRITE, MAP_SHARED, fd, 0);
  if (p == MAP_FAILED) {
    close(fd);
    return fail(HX_ENOMEM, "hx_shared_router_open: mmap failed");
  }
  auto* c = static_cast<SharedCounter*>(p);
  if (create) {
    c->n_blocks = n_blocks;
    c->next.store(0, std::memory_order_relaxed);
    std::atomic_thread_fence(std::memory_order_release);
    c->magic = kMagic;
  } else if (c->magic != kMagic || c->n_blocks != n_blocks) {
    munmap(p, sizeof(SharedCounter));
    close(fd);
    return fail(HX_EINVAL, "hx_shared_router_open: segment not created, or for another block count");
  }
  auto* r = new hx_shared_router();
  r->name = name;
  r->fd = fd;
  r->c = c;
  *out = r;
  return HX_OK;
}

int hx_shared_router_next(hx_shared_router* r, int64_t* block) {
  HX_REQUIRE(r && block, HX_EINVAL, "hx_shared_router_next: null argument");
  const int64_t b = r->c->next.fetch_add(1, std::memory_order_relaxed);
  *block = b < r->c->n_blocks ? b : -1;
  return HX_OK;
}

int hx_shared_router_reset(hx_shared_router* r) {
  HX_REQUIRE(r, HX_EINVAL, "hx_shared_router_reset: null router");
  r->c->next.store(0, std::memory_order_relaxed);
  return HX_OK;
}

int hx_shared_router_close(hx_shared_router* r, int unlink_name) {
  HX_REQUIRE(r, HX_EINVAL, "hx_shared_router_close: null router");
  munmap(r->c, sizeof(SharedCounter));
  close(r->fd);
  if (unlink_name) shm_unlink(r->name.c_str());
  delete r;
  return HX_OK;
}

}  // extern "C"
