#!/bin/bash
# SASS instruction count of each eval-kernel variant (code footprint; instruction fetch is the top stall).
# Usage: bash tools/sass_size.sh [-DEXTRA ...]
cd "$(dirname "$0")/../paper_conf_cluster_subdbn18_b200/csrc" || exit 1
/usr/local/cuda/bin/nvcc -gencode arch=compute_100a,code=sm_100a -O3 -std=c++17 -lineinfo --fmad=false \
  -Xcompiler -fPIC,-O2,-ffp-contract=off -I../../include -I. "$@" -cubin culi_kernels.cu -o /tmp/culi_kernels.cubin \
  -Xptxas -v 2>&1 | grep -A2 "Compiling entry function '_ZN4culi16culi_eval_kernel" | grep "registers\|spill" | paste - - 
nvdisasm /tmp/culi_kernels.cubin | awk '/^\.text\./{name=$0} /\/\*[0-9a-f]+\*\/ +[A-Z@]/{n[name]++} END{for (k in n) print n[k], k}' | sort -k2 | grep -i "eval_kernel\|fanout_kernel\|define"
