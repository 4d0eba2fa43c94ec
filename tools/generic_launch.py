"""One generic-path call (w = 65) on 256 MiB, for an ncu capture of k1_generic."""
import os, sys
import torch
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_fast_bhatotiarv12_b200 as pkg
x = torch.empty(256 << 20, dtype=torch.uint8, device="cuda")
pkg.synth_fill(x, 2)
ch = pkg.Chunker(pkg.Params(window=65))
assert ch.path == "generic"
print(ch.chunk(x).numel())
