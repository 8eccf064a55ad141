#!/bin/bash
# Build libtridiag.so of git revision $1 into ab/libtridiag_$2.so (A/B timing
# of two builds on one GPU box: TRIDIAG_LIB_AB=ab/libtridiag_$2.so).
set -e
rev=$1; tag=$2
root=$(cd "$(dirname "$0")/.." && pwd)
tmp=$(mktemp -d)
git -C "$root" archive "$rev" paper_conf_ppopp_zhangco10_b200 include | tar -x -C "$tmp"
(cd "$tmp" && python -c "from paper_conf_ppopp_zhangco10_b200 import build as b; b.build(force=True)" > /dev/null)
mkdir -p "$root/ab"
cp "$tmp/paper_conf_ppopp_zhangco10_b200/libtridiag.so" "$root/ab/libtridiag_$tag.so"
rm -rf "$tmp"
echo "$root/ab/libtridiag_$tag.so"
