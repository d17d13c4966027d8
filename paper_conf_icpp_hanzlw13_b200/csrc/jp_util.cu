// jp_util.cu -- host-side helpers shared by the launchers of libjp.so: the
// once-per-(kernel, device) shared-memory attribute and the phase trace.
#include <chrono>
#include <cstdio>
#include <cstdlib>
#include <mutex>
#include <vector>
#include "jp_host.h"

namespace jp {

// host-side phase trace of the schedulers (JP_HOST_TRACE=1: microseconds since the previous mark, stderr)
void htrace(const char *what) {
  static const bool on = getenv("JP_HOST_TRACE") != nullptr;
  if (!on) return;
  thread_local auto prev = std::chrono::steady_clock::now();
  const auto now = std::chrono::steady_clock::now();
  fprintf(stderr, "[jp host] %-16s +%.1f us\n", what, std::chrono::duration<double, std::micro>(now - prev).count());
  prev = now;
}

cudaError_t set_smem_once(const void *fn, int bytes) {
  struct Ent { const void *fn; int dev, bytes; };
  static std::mutex mu;
  static std::vector<Ent> done;
  int dev = 0;
  cudaGetDevice(&dev);
  {
    std::lock_guard<std::mutex> g(mu);
    for (const Ent &e : done)
      if (e.fn == fn && e.dev == dev && e.bytes >= bytes) return cudaSuccess;
  }
  const cudaError_t e = cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, bytes);
  if (e == cudaSuccess) {
    std::lock_guard<std::mutex> g(mu);
    done.push_back({fn, dev, bytes});
  }
  return e;
}

}  // namespace jp
