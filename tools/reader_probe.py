"""Device reader probe: device read time / GB/s of the text vs the host reader, per config."""
import sys
import time

import torch

sys.path.insert(0, ".")
from paper_conf_cluster_subdbn18_b200 import culi  # noqa: E402
from paper_conf_cluster_subdbn18_b200 import workloads as W  # noqa: E402

def main():
  culi.load()
  import os
  sel = os.environ.get("PROBE", "C1,C3,C4,C5-1M").split(",")
  mk = {"C1": lambda: W.c1(), "C3": lambda: W.c3(), "C4": lambda: W.c4(), "C5-1M": lambda: W.c5(1 << 20),
        "C5-4M": lambda: W.c5(1 << 22)}
  for name, wl in [(k, mk[k]()) for k in sel]:
      ctx = culi.Context(heap_nodes=1 << 28)
      text = wl.defs if name == "C3" else wl.forms
      if name != "C3" and wl.defs:
          ctx.define(wl.defs)
      b = text.encode()
      dev = torch.frombuffer(bytearray(b), dtype=torch.uint8).cuda()
      for _ in range(2):
          if name == "C3":
              ctx.define_text(dev)
          else:
              ctx.eval_text(dev)
      ms, items, nodes = ctx.last_read()
      t0 = time.perf_counter(); img = ctx.read(b); th = time.perf_counter() - t0
      print("%-6s %9d bytes %9d items %9d nodes  device read %.3f ms (%.1f GB/s of text)  host read %.1f ms"
            % (name, len(b), items, nodes, ms, len(b) / ms / 1e6, th * 1e3), flush=True)
      ctx.close()


if __name__ == "__main__":
    main()
