#!/bin/bash
# Build libgss.so variants for A/B timing: tools/build_variants.sh name1 "-DFOO=1" name2 "-DBAR=2" ...
# Results in variants/libgss_<name>.so (the default build is restored at the end).
set -e
cd "$(dirname "$0")/.."
mkdir -p variants
while [ $# -gt 1 ]; do
  NAME=$1; FL=$2; shift 2
  GSS_NVCC_EXTRA="$FL" python -c "from paper_conf_ipps_leischneros10_b200 import _build; _build.build(force=True)" > /dev/null
  cp paper_conf_ipps_leischneros10_b200/libgss.so variants/libgss_$NAME.so
  echo "built $NAME ($FL)"
done
python -c "from paper_conf_ipps_leischneros10_b200 import _build; _build.build(force=True)" > /dev/null
