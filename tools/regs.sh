#!/bin/bash
# registers / spills per kernel of one CUDA source (ptxas -v): tools/regs.sh tea_cheb_tb.cu [grep-pattern]
cd "$(dirname "$0")/../paper_conf_cluster_mcintosh_smithm17_b200/csrc"
NCCL=$(python -c "import nvidia.nccl;print(list(nvidia.nccl.__path__)[0])")
nvcc -O3 -std=c++17 -gencode arch=compute_100a,code=sm_100a -Xptxas -v $EXTRA -I../../include -I$NCCL/include -c "$1" -o /tmp/regs_$$.o 2>&1 \
 | awk '/Function properties for/ {name=$NF} /spill stores/ {sp=$5"/"$9} /Used [0-9]+ registers/ {print name, $5, "regs spill(st/ld B)", sp}' \
 | sed -E 's/^_ZN3tea[0-9]+//; s/EvPK[^ ]*//; s/EEv[^ ]*//' | grep -E "${2:-.}"
rm -f /tmp/regs_$$.o
